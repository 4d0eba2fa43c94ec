#!/bin/bash
mkdir -p gpurun_out
ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 2 -c 1 -o gpurun_out/prof_small python tools/small_launches.py > /dev/null 2>&1
ncu --set full --clock-control none -k regex:k1_generic -s 1 -c 1 -o gpurun_out/prof_generic python tools/variant_speed.py > /dev/null 2>&1
python tools/variant_speed.py 2>&1 | grep GB

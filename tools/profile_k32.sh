#!/bin/bash
mkdir -p gpurun_out
ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 3 -c 1 -o gpurun_out/prof_k32_$1 \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --no-extra --variant k32 > /dev/null 2>&1
echo done

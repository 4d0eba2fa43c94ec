#!/bin/bash
mkdir -p gpurun_out
ncu --set full --clock-control none --import-source on -k regex:k_hash_chunks -s 1 -c 1 -o gpurun_out/prof_hash_$1 \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu > /dev/null 2>&1
echo done

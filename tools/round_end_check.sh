#!/bin/bash
# What the driver runs at round end (GPU side), for a final check: tests, smoke, bench, reference.
mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -2
python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
python bench.py > gpurun_out/bench_final.json 2> gpurun_out/bench_final.err; tail -1 gpurun_out/bench_final.json | cut -c1-200
timeout 600 python bench.py --impl reference > gpurun_out/bench_ref.json 2>&1; tail -1 gpurun_out/bench_ref.json | cut -c1-200
bash tools/gpu_profile.sh r01k skip-tests > /dev/null 2>&1; echo profiled

#!/bin/bash
# GPU-box measurement script (run under gpurun): tests, bench line, ncu launch list, ncu full
# capture of the hot kernel.  Usage: bash tools/gpu_profile.sh <tag> [skip-tests]
TAG=${1:-rXX}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv
if [ "$2" != "skip-tests" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -15
fi
python bench.py 2>&1 | tail -3 > gpurun_out/bench_$TAG.json
cat gpurun_out/bench_$TAG.json
ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_$TAG.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --no-extra > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 3 -c 1 -o gpurun_out/prof_k1_$TAG \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --no-extra > gpurun_out/ncu_full_$TAG.log 2>&1
tail -2 gpurun_out/ncu_full_$TAG.log
# the summary and the traffic JSON from the SAME report (bench.py's roofline.traffic cites it)
python tools/ncu_summary.py gpurun_out/prof_k1_$TAG.ncu-rep > gpurun_out/k1_bulk_ncu_full_$TAG.txt 2>&1
python tools/ncu_traffic.py gpurun_out/prof_k1_$TAG.ncu-rep profiles/${TAG}_k1_bulk_ncu_full.txt > gpurun_out/k1_traffic_$TAG.json 2>&1
if [ "$3" == "k32" ]; then
  # the k <= 32 kernel on the sparse trinomial x^31+x^13+1 (K32T, bench k32t_variant)
  ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 3 -c 1 -o gpurun_out/prof_k1k32t_$TAG \
      python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --no-extra --variant k32t > /dev/null 2>&1
  python tools/ncu_summary.py gpurun_out/prof_k1k32t_$TAG.ncu-rep > gpurun_out/k32t_ncu_full_$TAG.txt 2>&1
fi
# f2: the batched SHA-256 launch (3 x 1 GiB, the bench's hash_sha256 value), same summary tool
ncu --set full --clock-control none --import-source on -k regex:k_hash_chunks -s 1 -c 1 -o gpurun_out/prof_hash_$TAG \
    python tools/hash_once.py > gpurun_out/ncu_hash_$TAG.log 2>&1
python tools/ncu_summary.py gpurun_out/prof_hash_$TAG.ncu-rep > gpurun_out/hash_ncu_full_$TAG.txt 2>&1

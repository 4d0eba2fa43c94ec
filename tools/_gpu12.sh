mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -q -x -k "size_bound_state" 2>&1 | tail -2
ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 20 -c 1 -o gpurun_out/prof_small_r02 python tools/small_profile.py > /dev/null 2>&1
python tools/ncu_summary.py gpurun_out/prof_small_r02.ncu-rep > gpurun_out/r02_k1_bulk_1mib_ncu_full.txt 2>&1
ncu --set full --clock-control none --import-source on -k regex:k_hash_chunks -s 1 -c 3 -o gpurun_out/prof_hash_r02 python tools/hash_speed.py > /dev/null 2>&1
python tools/ncu_summary.py gpurun_out/prof_hash_r02.ncu-rep > gpurun_out/r02_hash_ncu_full.txt 2>&1
ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/r02_bench_launches.csv python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --no-extra > /dev/null 2>&1
python tools/launch_sum.py gpurun_out/r02_bench_launches.csv

mkdir -p gpurun_out
python tools/cpu_rate_probe.py 2>&1 | tee gpurun_out/cpu_rate_probe.txt
timeout 900 python bench.py --impl reference > gpurun_out/bench_ref_r02.json 2>&1; tail -c 600 gpurun_out/bench_ref_r02.json
bash tools/gpu_profile.sh r02 skip-tests > gpurun_out/gpu_profile_r02.log 2>&1; tail -5 gpurun_out/gpu_profile_r02.log

bash tools/sanitize.sh > gpurun_out/g5_sanitize.txt 2>&1
bash tools/gpu_profile.sh r02 skip-tests k32 > gpurun_out/g5_profile.txt 2>&1
timeout 600 python bench.py --impl reference > gpurun_out/g5_ref.json 2>&1

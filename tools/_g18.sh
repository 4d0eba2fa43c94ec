mkdir -p gpurun_out; rm -f gpurun_out/g18.txt
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "bounded or walk or adversarial or phase or one_cta" 2>&1 | tail -2 > gpurun_out/g18_tests.txt
python tools/walk_speed.py >> gpurun_out/g18.txt 2>&1
for n in 1048576 4194304 16000000; do python tools/bounded_small.py $n >> gpurun_out/g18.txt 2>&1; done
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -2 >> gpurun_out/g18_tests.txt
python tests/sanitize_cases.py >> gpurun_out/g18_tests.txt 2>&1

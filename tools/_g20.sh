mkdir -p gpurun_out; rm -f gpurun_out/g20.txt
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "bounded or walk or adversarial or phase or one_cta" 2>&1 | tail -2 > gpurun_out/g20_tests.txt
python tools/walk_speed.py >> gpurun_out/g20.txt 2>&1
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -2 >> gpurun_out/g20_tests.txt
python tests/sanitize_cases.py >> gpurun_out/g20_tests.txt 2>&1

mkdir -p gpurun_out; rm -f gpurun_out/g25.txt
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fuzz.py -q -x -k "long_window or funnel or random_case" 2>&1 | tail -2 > gpurun_out/g25_tests.txt
python tools/window_speed.py 48 65 80 96 128 129 256 1000 4096 > gpurun_out/g25.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -2 >> gpurun_out/g25_tests.txt
python tests/sanitize_cases.py >> gpurun_out/g25_tests.txt 2>&1

mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -q -x -k "long_window or funnel or lengths" 2>&1 | tail -3 > gpurun_out/g13_tests.txt
python tools/window_speed.py > gpurun_out/g13_speed.txt 2>&1
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -3 >> gpurun_out/g13_tests.txt
python tests/sanitize_cases.py >> gpurun_out/g13_tests.txt 2>&1

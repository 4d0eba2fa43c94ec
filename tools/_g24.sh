mkdir -p gpurun_out; rm -f gpurun_out/g24.txt
timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -2 > gpurun_out/g24_tests.txt
for n in 1048576 268435456 1073741824; do python tools/bounded_small.py $n >> gpurun_out/g24.txt 2>&1; done
python tools/walk_speed.py >> gpurun_out/g24.txt 2>&1

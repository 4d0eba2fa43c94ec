mkdir -p gpurun_out; rm -f gpurun_out/g17.txt
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "bounded or walk or adversarial or phase" 2>&1 | tail -3 > gpurun_out/g17_tests.txt
timeout 900 python -m pytest tests/test_gpu_dist.py tests/test_gpu_fuzz.py -q -x 2>&1 | tail -2 >> gpurun_out/g17_tests.txt
for v in "" _oldwalk; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/walk_speed.py >> gpurun_out/g17.txt 2>&1; done

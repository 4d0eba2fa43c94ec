mkdir -p gpurun_out; rm -f gpurun_out/g22.txt
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "bounded or walk or adversarial or phase or one_cta" 2>&1 | tail -1 > gpurun_out/g22_tests.txt
SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred_rep0.so timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "bounded or walk or adversarial or phase or one_cta" 2>&1 | tail -1 >> gpurun_out/g22_tests.txt
for v in "" _rep0 _rep1 _rep2; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/walk_speed.py >> gpurun_out/g22.txt 2>&1; done

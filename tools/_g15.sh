mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_config4.py -q -x 2>&1 | tail -3 > gpurun_out/g15_tests.txt
bash tools/bench_ab.sh _sbb8 > gpurun_out/g15_ab.txt 2>&1
for v in "" _sbb8; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/bounded_small.py 4194304 >> gpurun_out/g15_ab.txt 2>&1; done

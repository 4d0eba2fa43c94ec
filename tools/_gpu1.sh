set -x
free -g | head -2; nproc
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q --ignore=tests/test_gpu_fullsize.py 2>&1 | tail -8
for v in "" _nodefer; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so timeout 300 python tools/k32_speed.py; done 2>&1 | tee gpurun_out/k32_speed_a.txt

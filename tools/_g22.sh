for v in "" _wsb _wsb8 _wsb8s3; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so timeout 300 python tools/hash_speed.py 2>&1 | tail -1; done
SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred_wsb8.so timeout 900 python -m pytest tests/test_gpu_hash.py -q -x 2>&1 | tail -1

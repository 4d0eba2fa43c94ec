for v in "" _h2 "" _h2; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/hash_speed.py 2>&1 | tail -1; done

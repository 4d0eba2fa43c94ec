for v in "" _lea "" _lea; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/k32_speed.py 2>&1 | grep -v "le r=1\|deg 29\|30+x"; done

mkdir -p gpurun_out; rm -f gpurun_out/g23.txt
for v in "" _one1g; do for n in 67108864 268435456 1073741824; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/bounded_small.py $n >> gpurun_out/g23.txt 2>&1; done; done

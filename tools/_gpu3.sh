mkdir -p gpurun_out
for v in _hi _hinodefer; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so timeout 300 python tools/k32_speed.py 2>&1 | grep k32t; done | tee gpurun_out/k32_speed_d.txt
SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred_nodefer.so ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 2 -c 1 -o gpurun_out/prof_k32t_nodefer python tools/prof_one.py 0x80002001 > /dev/null 2>&1
python tools/ncu_summary.py gpurun_out/prof_k32t_nodefer.ncu-rep > gpurun_out/k32t_nodefer.txt 2>&1

mkdir -p gpurun_out
for v in "" _nodefer; do
  SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 2 -c 1 -o gpurun_out/prof_k32b$v python tools/prof_one.py > /dev/null 2>&1
  python tools/ncu_summary.py gpurun_out/prof_k32b$v.ncu-rep > gpurun_out/k32b$v.txt 2>&1
done
timeout 1200 python -m pytest tests/test_gpu_fullsize.py -x -q 2>&1 | tail -5

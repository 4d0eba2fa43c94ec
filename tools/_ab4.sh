mkdir -p gpurun_out; rm -f gpurun_out/ab4_k32.jsonl
for r in 1 2; do for v in "" _nopack; do
  SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/k32_speed.py >> gpurun_out/ab4_k32.jsonl 2>&1
done; done
timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -2 > gpurun_out/ab4_tests.txt

mkdir -p gpurun_out; rm -f gpurun_out/g16_ab.txt
bash tools/bench_ab.sh _sbb8 _sbb4 > gpurun_out/g16_ab.txt 2>&1
for v in "" _sbb8 _sbb4; do for n in 1048576 4194304 16000000 67108864; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python tools/bounded_small.py $n >> gpurun_out/g16_ab.txt 2>&1; done; done
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -3 > gpurun_out/g16_tests.txt
python tests/sanitize_cases.py >> gpurun_out/g16_tests.txt 2>&1

mkdir -p gpurun_out
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -2 > gpurun_out/g3_tests.txt
python bench.py > gpurun_out/g3_bench.json 2> gpurun_out/g3_bench.err
timeout 600 python bench.py --impl reference > gpurun_out/g3_ref.json 2>&1
ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 3 -c 1 -o gpurun_out/prof_k32t_g3 \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --no-extra --variant k32t > gpurun_out/g3_ncu.log 2>&1
python tools/ncu_summary.py gpurun_out/prof_k32t_g3.ncu-rep > gpurun_out/g3_k32t_summary.txt 2>&1

mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.draw --format=csv
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -3
python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
python bench.py > gpurun_out/bench_r02b.json 2> gpurun_out/bench_r02b.err; tail -1 gpurun_out/bench_r02b.json | head -c 600; echo
timeout 900 python bench.py --impl reference > gpurun_out/bench_ref_r02b.json 2>&1; tail -1 gpurun_out/bench_ref_r02b.json | head -c 300; echo

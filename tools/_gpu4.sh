mkdir -p gpurun_out
free -g | head -2
timeout 1500 python -m pytest tests -m gpu -x -q 2>&1 | tail -6
python bench.py > gpurun_out/bench_r02a.json 2> gpurun_out/bench_r02a.err; tail -c 3000 gpurun_out/bench_r02a.json
SHRED_BENCH_BACKEND=gloo SHRED_BENCH_DEVICE=0 SHRED_BENCH_STREAM=$((4<<30)) timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29533 bench.py --gpus 2 --steps 5 --warmup 3 > gpurun_out/bench_r02_n2.json 2> gpurun_out/bench_r02_n2.err; tail -c 1500 gpurun_out/bench_r02_n2.json; tail -5 gpurun_out/bench_r02_n2.err

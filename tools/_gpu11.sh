mkdir -p gpurun_out
bash tools/sanitize.sh 2>&1 | tee gpurun_out/sanitize_r02.txt
python bench.py --no-cpu --no-e2e --steps 10 > gpurun_out/bench_x.json 2>&1; python -c "
import json; d=json.loads(open('gpurun_out/bench_x.json').read().strip().splitlines()[-1]); print(d.get('config2_16gib_fed')); print(d.get('config4_sweep')); print(d.get('extra_error'))"

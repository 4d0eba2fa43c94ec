mkdir -p gpurun_out
timeout 1500 python -m pytest tests -m gpu -x -q 2>&1 | tail -3
python tools/host_overhead.py
python bench.py --no-cpu --no-e2e --steps 20 > gpurun_out/bench_w.json 2>&1; python -c "
import json; d=json.loads(open('gpurun_out/bench_w.json').read().strip().splitlines()[-1]); print('value', d['value'], 'k1', d['roofline']['achieved'], '1MiB', d['config1_1mib'], 'bounded', d['bounded_2048_65536']['value'], 'k32t', d['k32t_variant']['value'])"

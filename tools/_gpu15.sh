mkdir -p gpurun_out
python bench.py > gpurun_out/bench_r02d.json 2> gpurun_out/bench_r02d.err
timeout 900 python bench.py --impl reference > gpurun_out/bench_ref_r02d.json 2>&1
python -c "
import json; d=json.loads(open('gpurun_out/bench_r02d.json').read().strip().splitlines()[-1]); print('value', d['value'], 'k1', d['roofline']['achieved'], d['roofline']['frac'], 'k32t', d['k32t_variant']['value'], 'k63t', d['k63t_variant']['value'], 'k32b', d['k32_variant']['value'], '1MiB', d['config1_1mib'], 'hash', d['hash_sha256'], 'bounded', d['bounded_2048_65536']['value'], 'c3', d['config3_64gib']['value'], 'cpu', d['cpu_baseline']['value'], 'e2e', d['e2e']['value'], 'c2', d['config2_16gib_fed']['value'], [p['gbs'] for p in d['config4_sweep']['points']], d['config4_sweep']['pipeline_8k'], d['clocks'])"
tail -c 300 gpurun_out/bench_ref_r02d.json

mkdir -p gpurun_out


T0=$(date +%s); python bench.py > gpurun_out/bench_r02c.json 2> gpurun_out/bench_r02c.err; echo "bench wall $(( $(date +%s) - T0 )) s"
python -c "
import json; d=json.loads(open('gpurun_out/bench_r02c.json').read().strip().splitlines()[-1]); print('value', d['value'], 'k1', d['roofline']['achieved'], d['roofline']['frac'], 'k32t', d['k32t_variant']['value'], 'k63t', d['k63t_variant']['value'], 'k32b', d['k32_variant']['value'], '1MiB', d['config1_1mib'], 'hash', d['hash_sha256']['value'], 'bounded', d['bounded_2048_65536']['value'], 'c3', d['config3_64gib']['value'], 'cpu', d['cpu_baseline']['value'])"

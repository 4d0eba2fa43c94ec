mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_api.py -x -q 2>&1 | tail -3
for v in "" _nofuse; do SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so python bench.py --no-cpu --no-e2e --steps 20 > gpurun_out/bench_fuse$v.json 2>&1; python -c "
import json; d=json.loads(open('gpurun_out/bench_fuse$v.json').read().strip().splitlines()[-1]); print('$v value', d['value'], 'k1', d['roofline']['achieved'], 'share', d['roofline']['share_of_step'], '1MiB', d['config1_1mib']['us_per_call'], d['config1_1mib']['us_per_graph_replay'], 'bounded', d['bounded_2048_65536']['value'], 'launches', d['gpu_launches'])"; done

mkdir -p gpurun_out


T0=$(date +%s); python bench.py > gpurun_out/bench_r02c.json 2> gpurun_out/bench_r02c.err; echo "bench wall $(( $(date +%s) - T0 )) s"
python -c "
import json; d=json.loads(open('gpurun_out/bench_r02c.json').read().strip().splitlines()[-1]); print('value', d['value'], 'k1', d['roofline']['achieved'], d['roofline']['frac'], 'k32t', d['k32t_variant']['value'], 'k63t', d['k63t_variant']['value'], 'k32b', d['k32_variant']['value'], '1MiB', d['config1_1mib'], 'hash', d['hash_sha256']['value'], 'bounded', d['bounded_2048_65536']['value'], 'c3', d['config3_64gib']['value'], 'cpu', d['cpu_baseline']['value'])"
bash tools/gpu_profile.sh r02b skip-tests > gpurun_out/gpu_profile_r02b.log 2>&1; cat gpurun_out/k1_bulk_ncu_full_r02b.txt
ncu -i gpurun_out/prof_k1_r02b.ncu-rep --page raw --csv 2>/dev/null | python3 -c "
import csv,sys
rows=list(csv.reader(sys.stdin)); h,u,v=rows[0],rows[1],rows[2]
for i,k in enumerate(h):
    if ('warps_issue_stalled' in k and 'ratio' in k) or 'fmaheavy_cycles_active.avg' in k or 'alu_cycles_active.avg' in k:
        try:
            if float(v[i].replace(',',''))>0.02: print(k.replace('smsp__average_warps_issue_stalled_',''), v[i])
        except: pass
"

#!/bin/bash
# A/B of library builds on the bench's side lines: value, bounded mode, configs[0] latency, e2e.
# Usage (GPU box): bash tools/bench_ab.sh _variant1 _variant2 ...  (libshred<suffix>.so in-tree)
for v in "" "$@"; do
  export SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so
  [ -f "$SHRED_LIB" ] || continue
  echo "== ${v:-base}"
  python bench.py --steps 10 --warmup 3 --no-cpu 2>/dev/null | tail -1 | python -c "
import json,sys; d=json.loads(sys.stdin.read())
print('  value', d['value'], 'kernel', d['roofline']['achieved'], 'bounded', d['bounded_2048_65536']['value'],
      '1MiB us', d['config1_1mib']['us_per_call'], 'e2e', d['e2e']['value'], 'k32', d['k32_variant']['value'])"
done

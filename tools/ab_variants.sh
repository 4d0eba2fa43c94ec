#!/bin/bash
# A/B the compile-time variants of libshred (built in-tree as libshred_<name>.so): a parity
# smoke per variant, then the hot-kernel rate for the paper params and the k32 variant.
mkdir -p gpurun_out
for v in "" "$@"; do
  export SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so
  [ -f "$SHRED_LIB" ] || continue
  echo "== variant '${v:-base}'"
  timeout 300 python -m pytest tests/test_gpu_parity.py -q -x -k "config1 or special or k32_path or bounded_variants or lengths" 2>&1 | tail -1
  for var in paper k32; do
    python bench.py --steps 50 --warmup 5 --no-e2e --no-cpu --no-extra --variant $var 2>/dev/null | tail -1 | \
      python -c "import json,sys; d=json.loads(sys.stdin.read()); print('  $var value', d['value'], 'kernel', d['roofline']['achieved'], 'GB/s', d['roofline']['avg_launch_ms'], 'ms', 'clk', d['clocks']['sm_mhz'])"
  done
done

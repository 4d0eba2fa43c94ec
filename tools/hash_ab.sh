#!/bin/bash
for v in "" "$@"; do
  export SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so
  echo "== ${v:-base}"
  python bench.py --steps 3 --warmup 3 --no-cpu --no-e2e 2>/dev/null | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); print(d['hash_sha256'])"
done

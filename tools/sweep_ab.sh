for v in _old _alu ""; do
  export SHRED_LIB=$PWD/paper_conf_fast_bhatotiarv12_b200/libshred$v.so
  echo "== ${v:-base}"
  python tools/sweep.py 2>&1 >/dev/null | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l)
        if d['D'] in (2048, 8192, 65536): print(' D',d['D'],'on' if d['bounds']!='off' else 'off','gbs',d['gbs'],'pipe',d['pipeline_gbs'],'batched',d['pipeline_batched_gbs'])"
done

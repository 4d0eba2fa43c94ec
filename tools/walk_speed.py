"""Bounded-mode call time on 1 GiB when the speculative size rule falls back to its serial walk
(min >> D: blocks of 16 candidates rarely re-sync) vs the usual LBFS bounds."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

n = 1 << 30
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
out = torch.empty(n // 256, dtype=torch.int64, device="cuda")
c = torch.zeros(1, dtype=torch.int64, device="cuda")
for mn, mx in ((2048, 65536), (8192, 65536), (32768, 0), (65536, 0), (131072, 262144)):
    ch = pkg.Chunker(pkg.Params(min_size=mn, max_size=mx))
    ch.chunk_async(x, out, c)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(3):
        ch.chunk_async(x, out, c)
    e1.record()
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1) / 3
    print(json.dumps({"min": mn, "max": mx, "ms_per_call": round(ms, 3), "gbs": round(n / (ms * 1e-3) / 1e9, 1),
                      "cuts": int(c.item()), "lib": os.path.basename(os.environ.get("SHRED_LIB", "libshred.so"))}),
          flush=True)

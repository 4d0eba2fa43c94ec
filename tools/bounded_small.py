"""Device time per 1 MiB call, unbounded vs bounded (min 2048 / max 65536), from 20 calls captured
in one CUDA graph (no host enqueue cost), per library build (SHRED_LIB selects an A/B variant)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

n = int(sys.argv[1]) if len(sys.argv) > 1 else 1 << 20
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 1)
o = torch.empty(4096 + n // 256, dtype=torch.int64, device="cuda")
c = torch.zeros(1, dtype=torch.int64, device="cuda")
res = {"lib": os.path.basename(os.environ.get("SHRED_LIB", "libshred.so")), "bytes": n}
for name, p in (("unbounded", pkg.Params()), ("bounded", pkg.Params(min_size=2048, max_size=65536))):
    ch = pkg.Chunker(p)
    gs = torch.cuda.Stream()
    with torch.cuda.stream(gs):
        for _ in range(50):
            ch.chunk_async(x, o, c, stream=gs)
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=gs):
        for _ in range(20):
            ch.chunk_async(x, o, c, stream=gs)
    for _ in range(20):
        g.replay()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(50):
        g.replay()
    e1.record()
    torch.cuda.synchronize()
    res[name + "_us"] = round(e0.elapsed_time(e1) * 1e3 / 1000, 2)
    res[name + "_cuts"] = int(c.item())
print(json.dumps(res))

"""f2 A/B helper: SHA-256 of every chunk of the 1 GiB configs[1] base file (seed 2), one call per
buffer, bounds off and 2048/65536; batch of 3 if the library has shred_hash_chunks_batch."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

n = 1 << 30
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
res = {"lib": os.path.basename(os.environ.get("SHRED_LIB", "libshred.so"))}
for name, p in (("off", pkg.Params()), ("bounded", pkg.Params(min_size=2048, max_size=65536))):
    ch = pkg.Chunker(p)
    cuts = torch.empty(n // 1024, dtype=torch.int64, device="cuda")
    nc = torch.zeros(1, dtype=torch.int64, device="cuda")
    ch.chunk_async(x, cuts, nc)
    digs = [torch.empty((n // 1024 + 1) * 32, dtype=torch.uint8, device="cuda") for _ in range(3)]
    ch.hash_chunks_async(x, cuts, nc, digs[0])
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(3):
        ch.hash_chunks_async(x, cuts, nc, digs[0])
    e1.record()
    torch.cuda.synchronize()
    res[name] = round(3 * n / (e0.elapsed_time(e1) * 1e-3) / 1e9, 1)
    if hasattr(pkg.lib(), "shred_hash_chunks_batch"):
        try:
            ch.hash_chunks_batch_async([(x, cuts, nc, d) for d in digs])
            torch.cuda.synchronize()
            e0.record()
            ch.hash_chunks_batch_async([(x, cuts, nc, d) for d in digs])
            e1.record()
            torch.cuda.synchronize()
            res[name + "_batch3"] = round(3 * n / (e0.elapsed_time(e1) * 1e-3) / 1e9, 1)
        except Exception as e:
            res[name + "_batch3"] = repr(e)[:80]
print(json.dumps(res))

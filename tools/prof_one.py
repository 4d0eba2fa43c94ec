"""One-case driver for ncu captures: 1 GiB (seed 2) chunked 4 times with the given polynomial
(default: the deg-32 K32B instance).  Usage: python tools/prof_one.py [poly] [n_log2]"""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

poly = int(sys.argv[1], 0) if len(sys.argv) > 1 else 0x104C11DB7
n = 1 << (int(sys.argv[2]) if len(sys.argv) > 2 else 30)
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
ch = pkg.Chunker(pkg.Params(poly=poly))
out = torch.empty(n // 512 + 4096, dtype=torch.int64, device="cuda")
nn = torch.zeros(1, dtype=torch.int64, device="cuda")
for _ in range(4):
    ch.chunk_async(x, out, nn)
torch.cuda.synchronize()
print("cands", int(nn.item()), "path", ch.path)

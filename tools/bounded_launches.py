"""Bounded-mode launches on 1 GiB (for an ncu launch list)."""
import os, sys
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg
x = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
ch = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536))
out = torch.empty(1 << 20, dtype=torch.int64, device="cuda"); n = torch.zeros(1, dtype=torch.int64, device="cuda")
for _ in range(3):
    ch.chunk_async(x, out, n)
torch.cuda.synchronize()
print(int(n.item()))

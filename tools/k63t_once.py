"""One 1 GiB call with the sparse degree-63 trinomial x^63+x^11+1 (K63T): for ncu."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

x = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
ch = pkg.Chunker(pkg.Params(poly=0x8000000000000801))
out = torch.empty((1 << 30) // 512, dtype=torch.int64, device="cuda")
n = torch.zeros(1, dtype=torch.int64, device="cuda")
for _ in range(3):
    ch.chunk_async(x, out, n)
torch.cuda.synchronize()
print(ch.mode, int(n.item()))

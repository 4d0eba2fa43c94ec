"""configs[0] (1 MiB) calls for an ncu launch list / capture: 30 back-to-back shred_chunk calls."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

x = torch.empty(1 << 20, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 1)
ch = pkg.Chunker(pkg.Params())
o = torch.empty(4096, dtype=torch.int64, device="cuda")
n = torch.zeros(1, dtype=torch.int64, device="cuda")
for _ in range(30):
    ch.chunk_async(x, o, n)
torch.cuda.synchronize()
print("candidates", int(n.item()))

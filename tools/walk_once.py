"""One bounded 1 GiB call with min >> D (the size rule's serial walk): for an ncu launch list."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

mn = int(sys.argv[1]) if len(sys.argv) > 1 else 65536
x = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
ch = pkg.Chunker(pkg.Params(min_size=mn))
out = torch.empty(1 << 22, dtype=torch.int64, device="cuda")
c = torch.zeros(1, dtype=torch.int64, device="cuda")
for _ in range(2):
    ch.chunk_async(x, out, c)
torch.cuda.synchronize()
print(int(c.item()))

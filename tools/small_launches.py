"""A few back-to-back 1 MiB shred_chunk calls (paper params): the launch list of one call under
ncu (`ncu --metrics gpu__time_duration.sum ... python tools/small_launches.py`)."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

n = int(sys.argv[1]) if len(sys.argv) > 1 and sys.argv[1].isdigit() else 1 << 20
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 1)
ch = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536) if "--bounded" in sys.argv else pkg.Params())
o = torch.empty(4096 + n // 1024, dtype=torch.int64, device="cuda")
c = torch.zeros(1, dtype=torch.int64, device="cuda")
for _ in range(5):
    ch.chunk_async(x, o, c)
torch.cuda.synchronize()

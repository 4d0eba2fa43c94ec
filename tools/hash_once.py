"""f2 launches for an ncu capture: SHA-256 of every chunk of the 1 GiB configs[1] base file
(seed 2, paper parameters, bounds off), once as one buffer, then 3 x the buffer as one batch
(the bench's hash_sha256 value).  Select with ncu -k regex:k_hash_chunks -s 0|1 -c 1."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

n = 1 << 30
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
ch = pkg.Chunker(pkg.Params())
cuts = torch.empty(n // 1024, dtype=torch.int64, device="cuda")
nc = torch.zeros(1, dtype=torch.int64, device="cuda")
ch.chunk_async(x, cuts, nc)
digs = [torch.empty((n // 1024 + 1) * 32, dtype=torch.uint8, device="cuda") for _ in range(3)]
ch.hash_chunks_async(x, cuts, nc, digs[0])
ch.hash_chunks_batch_async([(x, cuts, nc, d) for d in digs])
torch.cuda.synchronize()
print("chunks", int(nc.item()) + 1)

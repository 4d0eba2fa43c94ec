"""Hot-kernel and call throughput by window length on 1 GiB (device-resident, paper polynomial
and K32T x^31+x^13+1, D = 8192): w <= 64 pops from the register ring, w > 64 from the second TMA
tile (long windows).  One JSON line per case; SHRED_LIB selects an A/B build."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

n = 1 << 30
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
out = torch.empty(n // 512, dtype=torch.int64, device="cuda")
nn = torch.zeros(1, dtype=torch.int64, device="cuda")
ws = [int(a) for a in sys.argv[1:]] or [48, 64, 65, 80, 96, 128, 129, 256, 1000, 4096]
for poly, name in ((pkg.Params().poly, "k63"), (0x80002001, "k32t")):
    for w in ws:
        ch = pkg.Chunker(pkg.Params(poly=poly, window=w))
        for _ in range(3):
            ch.chunk_async(x, out, nn)
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        ch.profile(True)
        e0.record()
        reps = 5
        for _ in range(reps):
            ch.chunk_async(x, out, nn)
        e1.record()
        torch.cuda.synchronize()
        ch.profile(False)
        kms, kn, kb = ch.profile_read()
        print(json.dumps({"poly": name, "window": w, "path": ch.path,
                          "call_gbs": round(reps * n / (e0.elapsed_time(e1) * 1e-3) / 1e9, 1),
                          "k1_gbs": round(kb / (kms * 1e-3) / 1e9, 1) if kms else None, "cands": int(nn.item())}),
              flush=True)

"""Hot-kernel throughput of the u32-state and u64-state paths on 1 GiB (device-resident), per
library build (SHRED_LIB=... selects an A/B variant).  Prints one JSON line per case:
the one-shot call (k1_bulk + k_scatter) and the k1_bulk launch alone (library events)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

n = 1 << 30
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
cases = {"k32t (x^31+x^13+1)": pkg.Params(poly=0x80002001),
         "k32t (x^30+x^21+1)": pkg.Params(poly=0x40200001),
         "k32t le r=1": pkg.Params(poly=0x80002001, marker=1, magic=1),
         "k32b (0x104C11DB7)": pkg.Params(poly=0x104C11DB7),
         "k32 (deg 29)": pkg.Params(poly=0x20000005 if len(sys.argv) < 2 else int(sys.argv[1], 0)),
         "k32b le r=1": pkg.Params(poly=0x104C11DB7, marker=1, magic=1),
         "k63 (paper)": pkg.Params(),
         "k63t (x^63+x^11+1)": pkg.Params(poly=0x8000000000000801)}
out = torch.empty(n // 512, dtype=torch.int64, device="cuda")
nn = torch.zeros(1, dtype=torch.int64, device="cuda")
for name, p in cases.items():
    try:
        ch = pkg.Chunker(p)
    except Exception as e:
        print(json.dumps({"case": name, "error": repr(e)}))
        continue
    for _ in range(3):
        ch.chunk_async(x, out, nn)
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    ch.profile(True)
    e0.record()
    reps = 10
    for _ in range(reps):
        ch.chunk_async(x, out, nn)
    e1.record()
    torch.cuda.synchronize()
    ch.profile(False)
    kms, kn, kb = ch.profile_read()
    print(json.dumps({"case": name, "path": ch.path, "mode": ch.mode, "call_gbs": round(reps * n / (e0.elapsed_time(e1) * 1e-3) / 1e9, 1),
                      "k1_gbs": round(kb / (kms * 1e-3) / 1e9, 1), "cands": int(nn.item()),
                      "lib": os.path.basename(os.environ.get("SHRED_LIB", "libshred.so"))}), flush=True)

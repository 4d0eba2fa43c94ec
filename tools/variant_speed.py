"""Throughput of the kernel paths for parameter variants (256 MiB device-resident)."""
import os, sys
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg

n = 256 << 20
x = torch.empty(n, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
cases = {"paper (k63 eq pow2)": pkg.Params(), "k32": pkg.Params(poly=0x104C11DB7),
         "le marker": pkg.Params(divisor=8192, magic=1, marker=1), "w=32": pkg.Params(window=32),
         "w=64": pkg.Params(window=64), "D=10000": pkg.Params(divisor=10000, magic=7),
         "deg 40": pkg.Params(poly=0x10000000039), "w=47": pkg.Params(window=47),
         "w=31 k32": pkg.Params(poly=0x104C11DB7, window=31), "w=5": pkg.Params(window=5),
         "w=65": pkg.Params(window=65), "w=47 le": pkg.Params(window=47, divisor=8192, magic=1, marker=1),
         "deg 8": pkg.Params(poly=0x11D, divisor=256, magic=7),
         "D=10000 le": pkg.Params(divisor=10000, magic=1, marker=1),
         "D=2^40 le": pkg.Params(divisor=1 << 40, magic=1 << 27, marker=1),
         "D=3*2^32 eq": pkg.Params(divisor=3 << 32, magic=12345),
         "k32 D=1000 le": pkg.Params(poly=0x104C11DB7, divisor=1000, magic=0, marker=1)}
out = torch.empty(n // 256, dtype=torch.int64, device="cuda"); nn = torch.zeros(1, dtype=torch.int64, device="cuda")
for name, p in cases.items():
    try:
        ch = pkg.Chunker(p)
    except Exception as e:
        print(name, "init failed", e); continue
    ch.chunk_async(x, out, nn); torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(3):
        ch.chunk_async(x, out, nn)
    e1.record(); torch.cuda.synchronize()
    print(f"{name:22s} path={ch.path:8s} {3 * n / (e0.elapsed_time(e1) * 1e-3) / 1e9:9.1f} GB/s")

import os, sys, json, torch
sys.path.insert(0, '/root/repo')
import paper_conf_fast_bhatotiarv12_b200 as pkg
n = 1 << 30
x = torch.empty(n, dtype=torch.uint8, device="cuda"); pkg.synth_fill(x, 2)
ch = pkg.Chunker(pkg.Params())
cuts = torch.empty(n // 1024, dtype=torch.int64, device="cuda"); nc = torch.zeros(1, dtype=torch.int64, device="cuda")
ch.chunk_async(x, cuts, nc)
dig = torch.empty((n // 1024 + 1) * 32, dtype=torch.uint8, device="cuda")
ch.hash_chunks_async(x, cuts, nc, dig); torch.cuda.synchronize()
ev = [torch.cuda.Event(enable_timing=True) for _ in range(7)]
ev[0].record()
for k in range(6):
    ch.hash_chunks_async(x, cuts, nc, dig); ev[k + 1].record()
torch.cuda.synchronize()
print(os.path.basename(os.environ.get("SHRED_LIB", "new")), [round(ev[k].elapsed_time(ev[k + 1]), 3) for k in range(6)])

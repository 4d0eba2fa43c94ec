"""Host enqueue cost of one shred_chunk call (configs[0], 1 MiB) vs its device time."""
import os
import sys
import time

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

x = torch.empty(1 << 20, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 1)
ch = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536) if "--bounded" in sys.argv else pkg.Params())
o = torch.empty(4096, dtype=torch.int64, device="cuda")
n = torch.zeros(1, dtype=torch.int64, device="cuda")
lib = pkg.lib()
st = torch.cuda.current_stream().cuda_stream
args = (ch._ctx, x.data_ptr(), x.numel(), o.data_ptr(), o.numel(), n.data_ptr(), st)
for _ in range(500):
    ch.chunk_async(x, o, n)
torch.cuda.synchronize()
for name, fn in (("python chunk_async", lambda: ch.chunk_async(x, o, n)),
                 ("ctypes shred_chunk", lambda: lib.shred_chunk(*args))):
    N = 2000
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    t0 = time.perf_counter()
    for _ in range(N):
        fn()
    t1 = time.perf_counter()
    e1.record()
    torch.cuda.synchronize()
    print(f"{name}: host {1e6 * (t1 - t0) / N:.2f} us/call, device span {1e3 * e0.elapsed_time(e1) / N:.2f} us/call")

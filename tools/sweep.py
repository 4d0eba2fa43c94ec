"""configs[4] sweep on one B200: expected chunk size D in {2..64} KiB, bounds off / on
(min = D/4, max = 8D), over 10 backup-style snapshots of a 1 GiB master (10 GiB per point).

Per point: device GB/s (CUDA events around the 10 shred_chunk calls), mean chunk size, the
fraction of chunks shared with the master (dedup context).  Writes one JSON list to stdout."""
import json
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402
import tools.snapshots as S  # noqa: E402


def main():
    n = int(os.environ.get("SWEEP_BYTES", 1 << 30))
    buf = torch.empty(n, dtype=torch.uint8, device="cuda")
    cap = n // 512 + 65536
    out = torch.empty(cap, dtype=torch.int64, device="cuda")
    nn = torch.zeros(1, dtype=torch.int64, device="cuda")
    res = []
    for D in (2048, 4096, 8192, 16384, 32768, 65536):
        for bounded in (False, True):
            mn, mx = (D // 4, 8 * D) if bounded else (0, 0)
            ch = pkg.Chunker(pkg.Params(divisor=D, min_size=mn, max_size=mx))
            ms, tot_cuts, shared = 0.0, 0, []
            master = None
            for s in range(10):
                segs = S.build_snapshot(buf, 6, s)
                ch.chunk_async(buf, out, nn)          # warm (and the cuts for the stats)
                torch.cuda.synchronize()
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record()
                ch.chunk_async(buf, out, nn)
                e1.record()
                torch.cuda.synchronize()
                ms += e0.elapsed_time(e1)
                k = int(nn.item())
                cuts = out[:k].cpu().numpy()
                tot_cuts += k
                if s == 0:
                    master = cuts
                else:
                    shared.append(S.shared_chunks(cuts, master, n, segs))
            res.append({"D": D, "bounds": [mn, mx] if bounded else "off", "gbs": round(10 * n / (ms * 1e-3) / 1e9, 1),
                        "mean_chunk": round(10 * n / (tot_cuts + 10), 1),
                        "shared_with_master": [round(x, 4) for x in shared]})
            print(json.dumps(res[-1]), file=sys.stderr, flush=True)
    print(json.dumps(res))


if __name__ == "__main__":
    main()

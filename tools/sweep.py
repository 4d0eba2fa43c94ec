"""configs[4] sweep on one B200: expected chunk size D in {2..64} KiB, bounds off / on
(min = D/4, max = 8D), over 10 backup-style snapshots of a 1 GiB master (10 GiB per point).

Per point: chunking GB/s (CUDA events around the 10 shred_chunk calls), the whole dedup
pipeline's GB/s (chunk -> SHA-256 per chunk -> index lookup/insert, all chained on the device:
SURVEY §8(f) f2/f3), the mean chunk size, and the dedup ratio (10 GiB / unique bytes) with the
per-snapshot new-byte fractions (the replacement probability p of each snapshot for context).
Also per point, `pipeline_batched_gbs`: the same pipeline over the 10 snapshots as ONE backup
stream (10 GiB in HBM, one chunk / hash / index call each).  SHA-256 is sequential inside a
chunk, so a hash launch lasts at least as long as its longest chunk (~D ln(#chunks) bytes);
batching spreads that latency over 10x more bytes (DESIGN.md §5b f2/f3).
Writes one JSON list to stdout and one line per point to stderr."""
import json
import os
import sys

import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402
import synthgen  # noqa: E402
import tools.snapshots as S  # noqa: E402


def main():
    n = int(os.environ.get("SWEEP_BYTES", 1 << 30))
    buf = torch.empty(n, dtype=torch.uint8, device="cuda")
    cap = n // 512 + 65536
    out = torch.empty(cap, dtype=torch.int64, device="cuda")
    nn = torch.zeros(1, dtype=torch.int64, device="cuda")
    dig = torch.empty(cap * 32, dtype=torch.uint8, device="cuda")
    # the batched stream: 10 snapshots back to back
    big = torch.empty(10 * n, dtype=torch.uint8, device="cuda")
    for s in range(10):
        S.build_snapshot(big[s * n:(s + 1) * n], 6, s)
    bcap = 10 * n // 512 + 65536
    bout = torch.empty(bcap, dtype=torch.int64, device="cuda")
    bnn = torch.zeros(1, dtype=torch.int64, device="cuda")
    bdig = torch.empty(bcap * 32, dtype=torch.uint8, device="cuda")
    res = []
    for D in (2048, 4096, 8192, 16384, 32768, 65536):
        for bounded in (False, True):
            mn, mx = (D // 4, 8 * D) if bounded else (0, 0)
            ch = pkg.Chunker(pkg.Params(divisor=D, min_size=mn, max_size=mx))
            ch.index_reset(10 * n // max(256, D // 2))
            ms_chunk, ms_pipe, tot_cuts, new_frac = 0.0, 0.0, 0, []
            for s in range(10):
                S.build_snapshot(buf, 6, s)
                ch.chunk_async(buf, out, nn)          # warm
                torch.cuda.synchronize()
                e0, e1, e2 = (torch.cuda.Event(enable_timing=True) for _ in range(3))
                before = ch.index_stats()["new_bytes"]
                e0.record()
                ch.chunk_async(buf, out, nn)
                e1.record()
                ch.hash_chunks_async(buf, out, nn, dig)
                ch.index_insert_async(dig, out, nn, n)
                e2.record()
                torch.cuda.synchronize()
                ms_chunk += e0.elapsed_time(e1)
                ms_pipe += e0.elapsed_time(e2)
                tot_cuts += int(nn.item())
                new_frac.append(round((ch.index_stats()["new_bytes"] - before) / n, 4))
            st = ch.index_stats()
            # batched: one backup stream of the 10 snapshots (fresh index, second run timed)
            for it in range(2):
                ch.index_reset(10 * n // max(256, D // 2))
                torch.cuda.synchronize()
                b0, b1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                b0.record()
                ch.chunk_async(big, bout, bnn)
                ch.hash_chunks_async(big, bout, bnn, bdig)
                ch.index_insert_async(bdig, bout, bnn, 10 * n)
                b1.record()
                torch.cuda.synchronize()
            ms_batched = b0.elapsed_time(b1)
            bst = ch.index_stats()
            res.append({"D": D, "bounds": [mn, mx] if bounded else "off",
                        "gbs": round(10 * n / (ms_chunk * 1e-3) / 1e9, 1),
                        "pipeline_gbs": round(10 * n / (ms_pipe * 1e-3) / 1e9, 1),
                        "pipeline_batched_gbs": round(10 * n / (ms_batched * 1e-3) / 1e9, 1),
                        "dedup_ratio_batched": round(10 * n / max(1, bst["new_bytes"]), 3),
                        "mean_chunk": round(10 * n / (tot_cuts + 10), 1),
                        "dedup_ratio": round(10 * n / max(1, st["new_bytes"]), 3),
                        "new_fraction_per_snapshot": new_frac,
                        "p_per_snapshot": list(synthgen.SNAPSHOT_P), "index_full": st["full"]})
            print(json.dumps(res[-1]), file=sys.stderr, flush=True)
    print(json.dumps(res))


if __name__ == "__main__":
    main()

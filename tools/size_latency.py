"""Per-call latency and rate of shred_chunk over input sizes (device-resident, paper params and
the k32 variant): the launch-shape switch (small shape below ~19 MB) shows up here.

Usage (GPU box): python tools/size_latency.py [--json out.jsonl] [--bounded]
"""
import argparse
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402

SIZES = [64 << 10, 256 << 10, 1 << 20, 4 << 20, 16 << 20, 19 << 20, 24 << 20, 64 << 20, 256 << 20]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--json", default=None)
    ap.add_argument("--bounded", action="store_true", help="also the size rule on (min 2048 / max 65536)")
    a = ap.parse_args()
    out = open(a.json, "w") if a.json else None
    cases = [("paper", pkg.Params()), ("k32", pkg.Params(poly=0x104C11DB7))]
    if a.bounded:
        cases.append(("paper_bounded", pkg.Params(min_size=2048, max_size=65536)))
    for name, p in cases:
        ch = pkg.Chunker(p)
        for n in SIZES:
            x = torch.empty(n, dtype=torch.uint8, device="cuda")
            pkg.synth_fill(x, 1)
            cap = max(4096, 4 * n // p.divisor + 64)
            o = torch.empty(cap, dtype=torch.int64, device="cuda")
            c = torch.zeros(1, dtype=torch.int64, device="cuda")
            reps = max(5, min(200, (1 << 30) // n))
            for _ in range(5):
                ch.chunk_async(x, o, c)
            torch.cuda.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            for _ in range(reps):
                ch.chunk_async(x, o, c)
            e1.record()
            torch.cuda.synchronize()
            us = e0.elapsed_time(e1) * 1e3 / reps
            rec = {"params": name, "bytes": n, "us_per_call": round(us, 2),
                   "gbs": round(n / (us * 1e-6) / 1e9, 1), "candidates": int(c.item())}
            print(json.dumps(rec))
            if out:
                out.write(json.dumps(rec) + "\n")
    if out:
        out.close()


if __name__ == "__main__":
    main()

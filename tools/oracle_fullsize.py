"""Write tests/golden/oracle_fullsize.json: the CPU oracle's results on the full-size
BASELINE.json configs, for exact (element-by-element, via per-GiB SHA-256 digests) parity tests
on the GPU (tests/test_gpu_fullsize.py).

Calls only oracle/ (R2 direct per-window reduction over 1 GiB host slices with a w-1 byte
overlap, oracle.candidates_stream; the min/max rule oracle.size_bound) and synthgen/ (inputs).
Nothing here comes from the CUDA path.

  configs[2]: 16 GiB = 2^34 bytes of SplitMix64 seed 4, paper parameters; bounds off and
              min 2048 / max 65536.
  configs[3]: 64 GiB = 2^36 bytes of SplitMix64 seed 5, paper parameters; bounds off and on
              (SURVEY §8(d) d1 row 4).

Usage: python tools/oracle_fullsize.py [--only configs2|configs3]   (~10 min on 8 cores)
"""
import argparse
import json
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import oracle  # noqa: E402

OUT = os.path.join(ROOT, "tests", "golden", "oracle_fullsize.json")
CONFIGS = {"configs2": (4, 1 << 34), "configs3": (5, 1 << 36)}


def run(name, seed, n):
    t0 = time.time()
    parts = []
    for a, b, c in oracle.candidates_stream(seed, n, oracle.Params()):
        parts.append(c)
        print(f"{name}: [{a >> 30}, {b >> 30}) GiB, {c.size} candidates, {time.time() - t0:.0f} s", flush=True)
    cand = np.concatenate(parts)
    cuts = oracle.size_bound(cand, n, 2048, 65536)
    return {"seed": seed, "n": n, "params": "P=0xbfe6b8a5bf378d83, w=48, D=8192, r=0x78",
            "generator": "synthgen SplitMix64 counter mode", "bucket": 1 << 30,
            "candidates": {"count": int(cand.size), "first": cand[:4].tolist(), "last": cand[-4:].tolist(),
                           "buckets": oracle.bucket_digests(cand, n)},
            "bounded_2048_65536": {"count": int(cuts.size), "first": cuts[:4].tolist(), "last": cuts[-4:].tolist(),
                                   "buckets": oracle.bucket_digests(cuts, n)},
            "oracle_seconds": round(time.time() - t0, 1)}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--only", choices=list(CONFIGS))
    args = ap.parse_args()
    res = {}
    if os.path.exists(OUT):
        with open(OUT) as f:
            res = json.load(f)
    res["_source"] = ("tools/oracle_fullsize.py: oracle R2 (oracle/rabin_oracle.c) over synthgen bytes; "
                      "digest = SHA-256 of the little-endian u64 offsets c with j GiB < c <= (j+1) GiB "
                      "(oracle.bucket_digests)")
    for name, (seed, n) in CONFIGS.items():
        if args.only and name != args.only:
            continue
        res[name] = run(name, seed, n)
        with open(OUT, "w") as f:
            json.dump(res, f, indent=1)
    print("wrote", OUT)


if __name__ == "__main__":
    main()

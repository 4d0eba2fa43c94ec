"""Write tests/golden/oracle_config4.json: the CPU oracle's results on BASELINE.json configs[4] at
full size -- 10 backup-style snapshots of a 1 GiB master (SplitMix64 seed 6, synthgen.snapshot's
recipe) chunked as one 10 GiB stream, D = 2, 4, 8, 16, 32, 64 KiB with r = 0x78, bounds off and
min D/4 / max 8D -- as per-GiB SHA-256 digests of the u64 offset lists, for exact parity tests on
the GPU (tests/test_gpu_config4.py).

Calls only oracle/ (R2 direct per-window reduction over 1 GiB slices with a w-1 byte overlap, as
oracle.candidates_stream; the min/max rule oracle.size_bound) and synthgen/ (inputs).  Nothing
here comes from the CUDA path.

Usage: python tools/oracle_config4.py   (~10 min on 8 cores)
"""
import json
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import oracle  # noqa: E402
import synthgen  # noqa: E402

OUT = os.path.join(ROOT, "tests", "golden", "oracle_config4.json")
GiB = 1 << 30
MASTER, NSNAP = 6, 10
DS = (2048, 4096, 8192, 16384, 32768, 65536)


def snapshot_fast(s: int, n: int = GiB, segment: int = 1 << 20) -> np.ndarray:
    """synthgen.snapshot(MASTER, n, s) built with the fast generator (same bytes)."""
    out = synthgen.random_bytes_fast(MASTER, n)
    if s:
        nseg = (n + segment - 1) // segment
        u = synthgen._uniform(1000 + s, nseg)
        for g in np.nonzero(u < synthgen.SNAPSHOT_P[s])[0]:
            a = int(g) * segment
            b = min(n, a + segment)
            out[a:b] = synthgen.random_bytes_fast(100 + s, b - a, a)
    return out


def snapshot_range(s: int, a: int, b: int, segment: int = 1 << 20) -> np.ndarray:
    """Bytes [a, b) of snapshot s (b - a small): master bytes with the replaced segments' bytes."""
    out = synthgen.random_bytes_fast(MASTER, b - a, a)
    if s:
        nseg = (GiB + segment - 1) // segment
        u = synthgen._uniform(1000 + s, nseg)
        for g in range(a // segment, (b - 1) // segment + 1):
            if u[g] < synthgen.SNAPSHOT_P[s]:
                x, y = max(a, g * segment), min(b, (g + 1) * segment)
                out[x - a:y - a] = synthgen.random_bytes_fast(100 + s, y - x, x)
    return out


def main():
    t0 = time.time()
    n = NSNAP * GiB
    k = 47                                      # w - 1
    cands = {D: [] for D in DS}
    head = np.zeros(0, np.uint8)
    for s in range(NSNAP):
        cur = snapshot_fast(s)
        nxt = snapshot_range(s + 1, 0, 1) if s + 1 < NSNAP else np.zeros(0, np.uint8)
        a, b = s * GiB, (s + 1) * GiB
        data = np.concatenate([head, cur, nxt])          # stream bytes [a - len(head), b + len(nxt))
        lo = a - head.size
        for D in DS:
            c = oracle.candidates(data, oracle.Params(divisor=D)) + np.uint64(lo)
            cands[D].append(c[(c > np.uint64(a)) & (c <= np.uint64(b))])
        head = cur[-k:].copy()
        del cur, data
        print(f"snapshot {s}: {time.time() - t0:.0f} s", flush=True)
    res = {"_source": ("tools/oracle_config4.py: oracle R2 (oracle/rabin_oracle.c) over synthgen bytes; "
                       "digest = SHA-256 of the little-endian u64 offsets c with j GiB < c <= (j+1) GiB "
                       "(oracle.bucket_digests)"),
           "master_seed": MASTER, "snapshots": NSNAP, "n": n,
           "params": "P=0xbfe6b8a5bf378d83, w=48, r=0x78; bounds: min D/4, max 8D", "points": {}}
    for D in DS:
        cand = np.concatenate(cands[D])
        cuts = oracle.size_bound(cand, n, D // 4, 8 * D)
        res["points"][str(D)] = {
            "off": {"count": int(cand.size), "first": cand[:4].tolist(), "last": cand[-4:].tolist(),
                    "buckets": oracle.bucket_digests(cand, n)},
            "on": {"count": int(cuts.size), "first": cuts[:4].tolist(), "last": cuts[-4:].tolist(),
                   "buckets": oracle.bucket_digests(cuts, n)}}
    res["oracle_seconds"] = round(time.time() - t0, 1)
    with open(OUT, "w") as f:
        json.dump(res, f, indent=1)
    print("wrote", OUT, res["oracle_seconds"], "s")


if __name__ == "__main__":
    main()

"""Device-side construction of the config-5 backup snapshots (bench/test helper).

Snapshot s of master seed M (synthgen.snapshot's recipe, built directly in HBM): the SplitMix64
stream M, with each 1 MiB segment g replaced - independently with probability SNAPSHOT_P[s] - by
the bytes [g MiB, (g+1) MiB) of stream 100+s.  The replaced-segment choice uses the same host
uniform draws as synthgen.snapshot, so both constructions give identical bytes."""
from __future__ import annotations

import numpy as np
import torch

import synthgen


def replaced_segments(length: int, s: int, segment: int = 1 << 20) -> np.ndarray:
    if s == 0:
        return np.zeros(0, dtype=np.int64)
    nseg = (length + segment - 1) // segment
    u = synthgen._uniform(1000 + s, nseg)
    return np.nonzero(u < synthgen.SNAPSHOT_P[s])[0]


def build_snapshot(buf: torch.Tensor, master_seed: int, s: int, segment: int = 1 << 20) -> np.ndarray:
    """Fill `buf` (CUDA uint8) with snapshot s; returns the replaced segment indices."""
    from paper_conf_fast_bhatotiarv12_b200 import synth_fill
    n = buf.numel()
    synth_fill(buf, master_seed, 0)
    segs = replaced_segments(n, s, segment)
    for g in segs:
        a = int(g) * segment
        b = min(n, a + segment)
        synth_fill(buf[a:b], 100 + s, a)
    return segs


def shared_chunks(cuts_s: np.ndarray, cuts_m: np.ndarray, n: int, segs: np.ndarray,
                  segment: int = 1 << 20) -> float:
    """Fraction of snapshot chunks that are byte-identical to a master chunk: same [start, end)
    in both chunk lists and no overlap with a replaced segment (exact for this generator)."""
    bs = np.concatenate([[0], cuts_s.astype(np.int64), [n]])
    bm = set(zip(np.concatenate([[0], cuts_m.astype(np.int64)]).tolist(),
                 np.concatenate([cuts_m.astype(np.int64), [n]]).tolist()))
    rep = np.zeros((n + segment - 1) // segment + 1, dtype=bool)
    rep[segs] = True
    same = 0
    for a, b in zip(bs[:-1].tolist(), bs[1:].tolist()):
        if (a, b) in bm and not rep[a // segment:(b - 1) // segment + 1].any():
            same += 1
    return same / max(1, len(bs) - 1)

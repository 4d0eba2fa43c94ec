"""configs[4] at full size on one B200, exact against the oracle: 10 backup-style snapshots of a
1 GiB master (SplitMix64 seed 6, synthgen.snapshot's recipe, built in HBM by tools/snapshots.py)
chunked as one 10 GiB stream, D = 2, 4, 8, 16, 32, 64 KiB, bounds off and min D/4 / max 8D --
the launch configuration of bench.py's config4_sweep.

The oracle's results (R2 over 1 GiB slices with a w-1 byte overlap, then the size rule) are stored
as per-GiB SHA-256 digests of the u64 offset lists in tests/golden/oracle_config4.json, written by
tools/oracle_config4.py (oracle/ and synthgen/ only); the GPU's lists are digested the same way,
so every offset is compared.  PAPER.md L1293-L1361 (Fig. 18, the backup snapshots), L259-L265
(the size rule)."""
import json
import os
import sys

import numpy as np
import pytest
import torch

import oracle

pytestmark = [pytest.mark.gpu, pytest.mark.slow]

GiB = 1 << 30
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
GOLD = os.path.join(ROOT, "tests", "golden", "oracle_config4.json")


@pytest.fixture(scope="module")
def pkg():
    import paper_conf_fast_bhatotiarv12_b200 as P
    return P


@pytest.fixture(scope="module")
def stream(pkg):
    sys.path.insert(0, os.path.join(ROOT, "tools"))
    import snapshots as SN
    free, _ = torch.cuda.mem_get_info()
    if free < 12 * GiB:
        pytest.skip("needs ~12 GiB of free HBM")
    big = torch.empty(10 * GiB, dtype=torch.uint8, device="cuda")
    for s in range(10):
        SN.build_snapshot(big[s * GiB:(s + 1) * GiB], 6, s)
    yield big
    del big
    torch.cuda.empty_cache()


@pytest.mark.parametrize("D", [2048, 4096, 8192, 16384, 32768, 65536])
def test_config4_snapshot_stream_exact(pkg, stream, D):
    with open(GOLD) as f:
        g = json.load(f)
    n = g["n"]
    assert n == stream.numel()
    for bnd in ("off", "on"):
        ref = g["points"][str(D)][bnd]
        p = pkg.Params(divisor=D, min_size=D // 4 if bnd == "on" else 0, max_size=8 * D if bnd == "on" else 0)
        got = pkg.Chunker(p).chunk(stream).cpu().numpy().astype(np.uint64)
        what = f"D={D} bounds {bnd}"
        assert got.size == ref["count"], f"{what}: {got.size} cuts, oracle {ref['count']}"
        assert got[:4].tolist() == ref["first"] and got[-4:].tolist() == ref["last"], what
        dig = oracle.bucket_digests(got, n)
        bad = [j for j, (a, b) in enumerate(zip(dig, ref["buckets"])) if a != b]
        assert not bad, f"{what}: GiB buckets {bad} differ from the oracle"

"""configs[4] shape on the GPU: the D sweep over backup-style snapshots, bounds on and off,
bit-exact vs the oracle (reduced size: 24 MiB master, snapshots 0, 3, 5, 9)."""
import numpy as np
import pytest
import torch

import oracle
import synthgen

pytestmark = pytest.mark.gpu


def test_device_snapshot_matches_host_recipe():
    import tools.snapshots as S
    n = (5 << 20) + 123
    buf = torch.empty(n, dtype=torch.uint8, device="cuda")
    for s in (0, 1, 5, 9):
        S.build_snapshot(buf, 6, s)
        assert np.array_equal(buf.cpu().numpy(), synthgen.snapshot(6, n, s))


@pytest.mark.parametrize("D", [2048, 8192, 65536])
def test_sweep_point_exact(D):
    import paper_conf_fast_bhatotiarv12_b200 as pkg
    import tools.snapshots as S
    n = 24 << 20
    buf = torch.empty(n, dtype=torch.uint8, device="cuda")
    for bounded in (False, True):
        mn, mx = (D // 4, 8 * D) if bounded else (0, 0)
        ch = pkg.Chunker(pkg.Params(divisor=D, min_size=mn, max_size=mx))
        p = oracle.Params(divisor=D, min_size=mn, max_size=mx)
        master = None
        for s in (0, 3, 5, 9):
            segs = S.build_snapshot(buf, 6, s)
            got = ch.chunk(buf).cpu().numpy().astype(np.uint64)
            exp = oracle.chunk(buf.cpu().numpy(), p)
            assert np.array_equal(got, exp), (D, bounded, s)
            lens = np.diff(np.concatenate([[0], got.astype(np.int64), [n]]))
            if not bounded:
                assert 0.7 * D < lens.mean() < 1.3 * D
            else:
                mean_exp = mn + D * (1 - np.exp(-(mx - mn) / D))
                assert abs(lens[:-1].mean() - mean_exp) / mean_exp < 0.1
                assert lens[:-1].min() >= mn and lens.max() <= mx
            if s == 0:
                master = got
            else:
                f = S.shared_chunks(got, master, n, segs)
                assert f > 1 - 2.5 * synthgen.SNAPSHOT_P[s] - 0.05

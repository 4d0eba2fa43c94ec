"""Multi-process (gloo, world size 2 and 3, CPU) tests of the sharding orchestration (dist.py).

The per-shard engine here is the CPU oracle (test infrastructure), so these tests pin the
host logic: shard bounds, halos, the count all-gather and global offsets (C2), the distributed
size rule ("chain") and the C3 gather — through both engine interfaces dist.chunk_sharded
accepts: the synchronous one and the asynchronous one the CUDA Chunker has (counts, entry and
exit states in tensors; an undersized candidate buffer redone exactly).  The CUDA engine itself
runs the same code in tests/test_gpu_dist.py (2-3 processes on one GPU).
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle
import synthgen


class OracleEngine:
    """Per-shard engine backed by the oracle (tests only)."""

    def __init__(self, params: oracle.Params, data: np.ndarray):
        self.params = params
        self.data = data

    def candidates_range(self, x, halo, start, total_len):
        xs = x.numpy()
        w = self.params.window
        fps = oracle.window_fps(xs, self.params)                  # fp_i for local i >= w-1
        i_loc = np.nonzero(fps % np.uint64(self.params.divisor) == np.uint64(self.params.magic))[0] + (w - 1)
        c = i_loc.astype(np.int64) + (start - halo) + 1           # absolute cut c = i + 1
        c = c[(c >= start + 1) & (c < total_len)]                 # window ends i >= start
        return torch.from_numpy(c)

    def size_bound_state(self, cands, end, fin, s, held):
        c, s2, h2 = oracle.size_bound_from(cands.numpy().astype(np.uint64), end, fin, s, held,
                                           self.params.min_size, self.params.max_size)
        return torch.from_numpy(c.astype(np.int64)), s2, h2

    def size_bound(self, cands, total_len):
        return torch.from_numpy(oracle.size_bound(cands.numpy().astype(np.uint64), total_len,
                                                  self.params.min_size, self.params.max_size).astype(np.int64))


class OracleAsyncEngine(OracleEngine):
    """The asynchronous engine interface of the CUDA Chunker (candidates_range_async,
    size_bound_state_dev: counts and entry/exit states in tensors, outputs into caller buffers),
    backed by the oracle on CPU tensors, so the CPU tests run chunk_sharded's device-style path
    (no host values between the chain's rounds) too."""

    def candidates_range_async(self, x, halo, start, total_len, out, n_out):
        c = self.candidates_range(x, halo, start, total_len)
        n_out[0] = c.numel()
        m = min(c.numel(), out.numel())
        out[:m] = c[:m]

    def size_bound_state_dev(self, cands, n_cand, end, fin, state_in, out, n_out, state_out):
        n = min(int(n_cand[0]), cands.numel())
        cuts, s2, h2 = self.size_bound_state(cands[:n], end, fin, int(state_in[0]), bool(state_in[1]))
        n_out[0] = cuts.numel()
        m = min(cuts.numel(), out.numel())
        out[:m] = cuts[:m]
        state_out[0] = s2
        state_out[1] = int(h2)


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n, seed, params, q, mode="chain", asyn=False):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_fast_bhatotiarv12_b200 import dist as sd
        data = synthgen.random_bytes(seed, n)
        start, end = sd.shard_bounds(n, world, rank, align=4096)
        halo = sd.halo_of(start, params.window)
        x = torch.from_numpy(synthgen.random_bytes(seed, end - start + halo, start - halo))
        assert np.array_equal(x.numpy(), data[start - halo:end])   # halo regenerated locally
        own = torch.from_numpy(data[start:end].copy())
        x2 = sd.exchange_halo(own, start, params.window)            # C1 over the process group
        assert np.array_equal(x2.numpy(), x.numpy())
        eng = (OracleAsyncEngine if asyn else OracleEngine)(params, data)
        res = sd.chunk_sharded(x, halo, start, n, eng, mode=mode, cap=64 if asyn else None)
        allc = sd.gather_all(res).numpy()
        q.put((rank, res.base, res.total, res.local.numpy().tolist(), allc.tolist(),
               None if res.cuts is None else res.cuts.numpy().tolist(), res.cut_base, res.rounds))
    finally:
        dist.destroy_process_group()


def _run(world, n, seed, params, mode="chain", asyn=False):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n, seed, params, q, mode, asyn)) for r in range(world)]
    for p in procs:
        p.start()
    out = [q.get(timeout=300) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    return sorted(out)


@pytest.mark.parametrize("world", [2, 3])
def test_sharded_unbounded_matches_whole_stream(world):
    n = (1 << 20) + 12345
    params = oracle.Params(divisor=1024)
    exp = oracle.candidates(synthgen.random_bytes(7, n), params).astype(np.int64).tolist()
    out = _run(world, n, 7, params)
    cat = []
    for rank, base, total, local, allc, cuts, cut_base, rounds in out:
        assert base == len(cat)
        assert total == len(exp)
        cat += local
        assert allc == exp
        assert cuts is None
    assert cat == exp


@pytest.mark.parametrize("world", [2, 3])
def test_sharded_unbounded_async_engine_overflow_redo(world):
    """The asynchronous path with a deliberately small candidate buffer (64 entries): the counts
    exchanged are the true ones, and reading `local` redoes the overflowed shard exactly."""
    n = (1 << 20) + 12345
    params = oracle.Params(divisor=1024)
    exp = oracle.candidates(synthgen.random_bytes(7, n), params).astype(np.int64).tolist()
    out = _run(world, n, 7, params, asyn=True)
    cat = []
    for rank, base, total, local, allc, cuts, cut_base, rounds in out:
        assert base == len(cat) and total == len(exp)
        cat += local
    assert cat == exp


@pytest.mark.parametrize("world,mode,asyn", [(2, "gather", False), (2, "chain", False), (3, "chain", False),
                                             (2, "chain", True), (3, "chain", True)])
def test_sharded_bounded_global_size_rule(world, mode, asyn):
    n = (1 << 20) + 999
    params = oracle.Params(divisor=512, min_size=128, max_size=4096)
    data = synthgen.random_bytes(9, n)
    exp = oracle.chunk(data, params).astype(np.int64).tolist()
    out = _run(world, n, 9, params, mode, asyn)
    if mode == "gather":
        for rank, base, total, local, allc, cuts, cut_base, rounds in out:
            assert cuts == exp
    else:
        cat = []
        for rank, base, total, local, allc, cuts, cut_base, rounds in out:
            assert cut_base == len(cat)
            assert rounds <= world
            cat += cuts
        assert cat == exp


def test_sharded_chain_adversarial_phase_lock():
    """Periodic candidates 2 bytes apart with min = 3: entry guesses are out of phase, so the
    chain needs extra rounds; the result is still exact."""
    n = 300000
    params = oracle.Params(divisor=8192, min_size=3, max_size=0)
    ctx = mp.get_context("spawn")
    data = synthgen.periodic(b"\x04\xd5", n)
    exp = oracle.chunk(data, params).astype(np.int64).tolist()
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker_periodic, args=(r, 3, port, n, params, q)) for r in range(3)]
    for p in procs:
        p.start()
    out = sorted(q.get(timeout=300) for _ in range(3))
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    cat = []
    for rank, cuts, cut_base in out:
        assert cut_base == len(cat)
        cat += cuts
    assert cat == exp


def _worker_periodic(rank, world, port, n, params, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_conf_fast_bhatotiarv12_b200 import dist as sd
        data = synthgen.periodic(b"\x04\xd5", n)
        start, end = sd.shard_bounds(n, world, rank, align=4096)
        halo = sd.halo_of(start, params.window)
        x = torch.from_numpy(data[start - halo:end].copy())
        res = sd.chunk_sharded(x, halo, start, n, OracleEngine(params, data), mode="chain")
        q.put((rank, res.cuts.numpy().tolist(), res.cut_base))
    finally:
        dist.destroy_process_group()


def test_shard_bounds_cover_the_stream():
    from paper_conf_fast_bhatotiarv12_b200 import dist as sd
    for n in (0, 1, 4095, 4096, 10 ** 6, 64 << 30):
        for world in (1, 2, 3, 8):
            spans = [sd.shard_bounds(n, world, r) for r in range(world)]
            assert spans[0][0] == 0 and spans[-1][1] == n
            for (a, b), (c, d) in zip(spans, spans[1:]):
                assert b == c and a <= b
            for a, _ in spans:
                assert sd.halo_of(a) == min(47, a)

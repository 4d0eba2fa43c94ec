"""dist.chunk_sharded with the CUDA engine (the product path): 2-3 processes sharing cuda:0 over a
gloo process group (NCCL cannot put two ranks on one device; gloo stages the 8-16 byte exchanges
through host memory).  Unbounded (no host synchronisation inside chunk_sharded), the distributed
size rule ("chain", device-resident entry/exit states) and the C3 gather, each against the
oracle on the whole stream (partitions with a window overlap).
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

pytestmark = pytest.mark.gpu


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n, seed, kw, mode, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import paper_conf_fast_bhatotiarv12_b200 as pkg
        from paper_conf_fast_bhatotiarv12_b200 import dist as sd
        torch.cuda.set_device(0)
        ch = pkg.Chunker(pkg.Params(**kw), device=0)
        start, end = sd.shard_bounds(n, world, rank)
        halo = sd.halo_of(start, ch.params.window)
        x = torch.empty(end - start + halo, dtype=torch.uint8, device="cuda")
        pkg.synth_fill(x, seed, start - halo)                     # the shard with its halo, on device
        res = sd.chunk_sharded(x, halo, start, n, ch, mode=mode)
        out = {"base": res.base, "total": res.total, "local": res.local.cpu().numpy().tolist(),
               "rounds": res.rounds, "cut_base": res.cut_base,
               "cuts": None if res.cuts is None else res.cuts.cpu().numpy().tolist(),
               "device": res.local.device.type}
        q.put((rank, out))
    finally:
        dist.destroy_process_group()


def _run(world, n, seed, kw, mode="chain"):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n, seed, kw, mode, q)) for r in range(world)]
    for p in procs:
        p.start()
    out = sorted(q.get(timeout=600) for _ in range(world))
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    return [o for _, o in out]


@pytest.mark.parametrize("world", [2, 3])
def test_unbounded_cuda_engine(world):
    n = (24 << 20) + 12345
    exp = oracle.candidates(synthgen.random_bytes_fast(21, n), oracle.Params()).astype(np.int64).tolist()
    out = _run(world, n, 21, {})
    cat = []
    for o in out:
        assert o["device"] == "cuda" and o["base"] == len(cat) and o["total"] == len(exp)
        cat += o["local"]
    assert cat == exp


@pytest.mark.parametrize("world,mode", [(2, "chain"), (3, "chain"), (3, "gather")])
def test_bounded_cuda_engine(world, mode):
    n = (16 << 20) + 999
    kw = dict(min_size=2048, max_size=65536)
    exp = oracle.chunk(synthgen.random_bytes_fast(22, n), oracle.Params(**kw)).astype(np.int64).tolist()
    out = _run(world, n, 22, kw, mode)
    if mode == "gather":
        for o in out:
            assert o["cuts"] == exp
        return
    cat = []
    for o in out:
        assert o["cut_base"] == len(cat) and 1 <= o["rounds"] <= world
        cat += o["cuts"]
    assert cat == exp


def test_bounded_chain_phase_locked_needs_more_rounds():
    """Small D with min > 2 candidate gaps: entry guesses out of phase; exact after <= G rounds."""
    n = (4 << 20) + 77
    kw = dict(divisor=64, magic=5, min_size=200, max_size=0)
    exp = oracle.chunk(synthgen.random_bytes_fast(23, n), oracle.Params(**kw)).astype(np.int64).tolist()
    out = _run(3, n, 23, kw)
    cat = []
    for o in out:
        assert o["cut_base"] == len(cat)
        cat += o["cuts"]
    assert cat == exp


def test_bench_strong_scaling_mode_two_ranks():
    """bench.py's N > 1 mode (configs[3] strong scaling) end to end with 2 ranks on one GPU
    (gloo, a 64 MiB stream instead of 64 GiB): one JSON line from rank 0 whose total candidate
    count equals the oracle's on that stream and whose t1 run (the whole stream on rank 0)
    finds the same count."""
    import json
    import subprocess
    import sys
    n = 64 << 20
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = dict(os.environ, SHRED_BENCH_BACKEND="gloo", SHRED_BENCH_DEVICE="0", SHRED_BENCH_STREAM=str(n))
    r = subprocess.run([sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2",
                        "--master-addr", "127.0.0.1", "--master-port", str(_free_port()),
                        os.path.join(root, "bench.py"), "--gpus", "2", "--steps", "3", "--warmup", "3",
                        "--no-e2e"], capture_output=True, text=True, env=env, cwd=root, timeout=600)
    assert r.returncode == 0, r.stderr[-2000:]
    line = json.loads([ln for ln in r.stdout.splitlines() if ln.startswith("{")][-1])
    exp = oracle.candidates(synthgen.random_bytes_fast(5, n), oracle.Params()).size
    assert line["n_gpus"] == 2 and line["scaling"] == "strong"
    assert line["candidates_total"] == exp and line["t1_candidates"] == exp
    assert line["value"] > 0 and line["gpu_launches"] > 0

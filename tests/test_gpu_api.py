"""The C-ABI contract on the GPU: capacity overflow in-band, sticky streaming error, reset,
pointer-kind checks, independent contexts, parameter validation."""
import ctypes

import numpy as np
import pytest
import torch

import oracle
import synthgen

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def pkg():
    import paper_conf_fast_bhatotiarv12_b200 as P
    return P


def test_capacity_overflow_reports_true_count(pkg):
    data = synthgen.random_bytes(21, 1 << 20)
    x = torch.from_numpy(data).cuda()
    ch = pkg.Chunker(pkg.Params(divisor=256))
    exp = oracle.candidates(data, oracle.Params(divisor=256))
    for cap in (1, 10, exp.size - 1, exp.size):
        out = torch.full((cap,), -1, dtype=torch.int64, device="cuda")
        n = torch.zeros(1, dtype=torch.int64, device="cuda")
        ch.chunk_async(x, out, n)
        assert int(n.item()) == exp.size                       # the TRUE count, in band
        assert np.array_equal(out.cpu().numpy().astype(np.uint64), exp[:cap])
    chb = pkg.Chunker(pkg.Params(divisor=256, min_size=64, max_size=1024))
    expb = oracle.chunk(data, oracle.Params(divisor=256, min_size=64, max_size=1024))
    out = torch.full((5,), -1, dtype=torch.int64, device="cuda")
    n = torch.zeros(1, dtype=torch.int64, device="cuda")
    chb.chunk_async(x, out, n)
    assert int(n.item()) == expb.size
    assert np.array_equal(out.cpu().numpy().astype(np.uint64), expb[:5])


def test_streaming_overflow_is_sticky_until_reset(pkg):
    data = synthgen.random_bytes(22, 1 << 20)
    ch = pkg.Chunker(pkg.Params(divisor=256))
    out = torch.empty(4, dtype=torch.int64, device="cuda")
    n = torch.zeros(1, dtype=torch.int64, device="cuda")
    ch.feed_async(torch.from_numpy(data).cuda(), out, n)
    torch.cuda.synchronize()
    assert int(n.item()) > 4
    with pytest.raises(pkg.ShredError, match="sticky"):
        ch.feed(torch.from_numpy(data[:100]).cuda())
    ch.reset()
    got = np.concatenate([ch.feed(torch.from_numpy(data).cuda()).cpu().numpy(), ch.flush().cpu().numpy()])
    assert np.array_equal(got.astype(np.uint64), oracle.candidates(data, oracle.Params(divisor=256)))


def test_pageable_host_input_rejected(pkg):
    ch = pkg.Chunker(pkg.Params())
    L = pkg.lib()
    buf = np.zeros(4096, np.uint8)
    out = torch.empty(16, dtype=torch.int64, device="cuda")
    n = torch.zeros(1, dtype=torch.int64, device="cuda")
    rc = L.shred_feed(ch._ctx, buf.ctypes.data, buf.size, out.data_ptr(), 16, n.data_ptr(),
                      torch.cuda.current_stream().cuda_stream)
    assert rc == -1
    assert b"page-locked" in L.shred_last_error(ch._ctx)


def test_halo_contract_of_candidates_range(pkg):
    ch = pkg.Chunker(pkg.Params())
    x = torch.zeros(1000, dtype=torch.uint8, device="cuda")
    with pytest.raises(pkg.ShredError, match="halo"):
        ch.candidates_range(x, 10, 5000, 100000)              # halo must be min(47, start)


def test_two_contexts_are_independent(pkg):
    d1, d2 = synthgen.random_bytes(23, 3 << 20), synthgen.random_bytes(24, 2 << 20)
    a = pkg.Chunker(pkg.Params())
    b = pkg.Chunker(pkg.Params(divisor=1024, min_size=256, max_size=8192))
    s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()
    x1, x2 = torch.from_numpy(d1).cuda(), torch.from_numpy(d2).cuda()
    o1 = torch.empty(10000, dtype=torch.int64, device="cuda"); n1 = torch.zeros(1, dtype=torch.int64, device="cuda")
    o2 = torch.empty(10000, dtype=torch.int64, device="cuda"); n2 = torch.zeros(1, dtype=torch.int64, device="cuda")
    torch.cuda.synchronize()
    for _ in range(3):
        a.chunk_async(x1, o1, n1, stream=s1)
        b.chunk_async(x2, o2, n2, stream=s2)
    torch.cuda.synchronize()
    e1 = oracle.chunk(d1, oracle.Params())
    e2 = oracle.chunk(d2, oracle.Params(divisor=1024, min_size=256, max_size=8192))
    assert np.array_equal(o1[:int(n1.item())].cpu().numpy().astype(np.uint64), e1)
    assert np.array_equal(o2[:int(n2.item())].cpu().numpy().astype(np.uint64), e2)


def test_init_validation_and_paths(pkg):
    with pytest.raises(pkg.ShredError):
        pkg.Chunker(pkg.Params(poly=(1 << 63) | 1))            # reducible
    with pytest.raises(pkg.ShredError):
        pkg.Chunker(pkg.Params(divisor=1, magic=0))             # D < 2
    with pytest.raises(pkg.ShredError):
        pkg.Chunker(pkg.Params(poly=0x104C11DB7, divisor=(1 << 33)))   # D > 2^deg
    with pytest.raises(pkg.ShredError):
        pkg.Chunker(pkg.Params(marker=2))
    assert pkg.Chunker(pkg.Params(divisor=3000)).path == 'k63'
    assert pkg.Chunker(pkg.Params(divisor=3000, magic=5, marker=1)).path == 'k63'   # MK_REM
    assert pkg.Chunker(pkg.Params(divisor=3 << 32)).path == 'k63'                   # MK_REM
    assert pkg.Chunker(pkg.Params()).path == "k63"
    assert pkg.Chunker(pkg.Params(poly=0x104C11DB7)).path == "k32"
    assert pkg.Chunker(pkg.Params(window=47)).path == "k63"
    assert pkg.Chunker(pkg.Params(window=47, marker=1)).path == "k63"
    assert pkg.Chunker(pkg.Params(window=65)).path == "k63"                       # long window
    assert pkg.Chunker(pkg.Params(window=4096)).path == "k63"
    ch = pkg.Chunker(pkg.Params(min_size=100))
    assert ch.max_cuts(1001) == 1000 // 100 + 1
    got = pkg._binding._Params()
    assert pkg.lib().shred_get_params(ch._ctx, ctypes.byref(got)) == 0 and got.min_size == 100


def test_profile_hook_counts_hot_launches(pkg):
    ch = pkg.Chunker(pkg.Params())
    x = torch.empty(64 << 20, dtype=torch.uint8, device="cuda")
    pkg.synth_fill(x, 3)
    ch.profile(True)
    ch.chunk(x); ch.chunk(x)
    ch.profile(False)
    ms, launches, nbytes = ch.profile_read()
    assert launches == 2 and ms > 0 and nbytes == 2 * x.numel()


def test_feed_edge_cases_mixed_sources_and_empty(pkg):
    """Zero-length feeds change nothing; device and pinned-host pieces can be mixed in one stream;
    an empty shard range yields no candidates."""
    n = (2 << 20) + 17
    data = synthgen.random_bytes(25, n)
    for p in (pkg.Params(divisor=1024), pkg.Params(divisor=1024, min_size=300, max_size=5000)):
        ch = pkg.Chunker(p)
        ch.set_ring(2, 1 << 19)
        outs = []
        a = 0
        for k, b in enumerate((0, 1000, 1000, 300000, 1500000, n)):
            piece = torch.from_numpy(data[a:b].copy())
            x = piece.cuda() if k % 2 else piece.pin_memory()
            outs.append(ch.feed(x).cpu().numpy())
            a = b
        outs.append(ch.feed(torch.zeros(0, dtype=torch.uint8).cuda()).cpu().numpy())
        outs.append(ch.flush().cpu().numpy())
        got = np.concatenate(outs).astype(np.uint64)
        exp = oracle.chunk(data, oracle.Params(divisor=1024, min_size=p.min_size, max_size=p.max_size))
        assert np.array_equal(got, exp)
    ch = pkg.Chunker(pkg.Params())
    x = torch.from_numpy(data[:47].copy()).cuda()
    assert ch.candidates_range(x, 47, 47, n).numel() == 0      # halo only, empty range


@pytest.mark.parametrize("bounded", [False, True])
def test_cuda_graph_capture_and_replay(pkg, bounded):
    """A shred_chunk call (after a warm-up call sized its scratch) can be captured into a CUDA
    graph and replayed: the launch-bound small-input case (configs[0]) without per-call launch
    overhead.  Replays on new bytes (same buffer) give the new exact result."""
    n = (1 << 20) + 77
    p = pkg.Params(min_size=2048, max_size=65536) if bounded else pkg.Params()
    ch = pkg.Chunker(p)
    x = torch.empty(n, dtype=torch.uint8, device="cuda")
    out = torch.empty(4096, dtype=torch.int64, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    pkg.synth_fill(x, 1)
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        ch.chunk_async(x, out, cnt, stream=s)                # warm-up: sizes the ctx scratch
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    with torch.cuda.graph(g, stream=s):
        ch.chunk_async(x, out, cnt, stream=s)
    op = oracle.Params(min_size=p.min_size, max_size=p.max_size)
    for seed in (1, 2, 3):
        pkg.synth_fill(x, seed)
        torch.cuda.synchronize()
        g.replay()
        torch.cuda.synchronize()
        k = int(cnt.item())
        exp = oracle.chunk(synthgen.random_bytes(seed, n), op)
        assert np.array_equal(out[:k].cpu().numpy().astype(np.uint64), exp)

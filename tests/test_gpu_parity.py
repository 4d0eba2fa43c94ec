"""GPU parity: the CUDA path (through the C ABI) vs the CPU oracle, element by element.

Bar: bit-exact (integer work).  Sizes span several tiles/rows and ragged tails; edge cases are
empty/short inputs, unaligned bases, adversarial candidate density (list overflow + re-roll),
all-zero / all-0xFF, and every kernel path (k63, k32, long windows, generic).
"""
import numpy as np
import pytest
import torch

import oracle
import synthgen

pytestmark = pytest.mark.gpu

LBFS = oracle.LBFS_POLY


@pytest.fixture(scope="module")
def pkg():
    import paper_conf_fast_bhatotiarv12_b200 as P
    return P


def dev(a: np.ndarray, offset: int = 0) -> torch.Tensor:
    """Copy to the GPU; `offset` > 0 returns a view starting `offset` bytes into a buffer."""
    buf = torch.empty(a.size + offset + 64, dtype=torch.uint8, device="cuda")
    t = buf[offset:offset + a.size]
    t.copy_(torch.from_numpy(a))
    return t


def oparams(p) -> oracle.Params:
    return oracle.Params(p.poly, p.window, p.divisor, p.magic, p.min_size, p.max_size, p.marker)


def check_chunk(ch, data: np.ndarray, offset: int = 0, method: int = 2):
    got = ch.chunk(dev(data, offset)).cpu().numpy().astype(np.uint64)
    exp = oracle.chunk(data, oparams(ch.params), method=method)
    assert got.size == exp.size, (got.size, exp.size)
    assert np.array_equal(got, exp)
    return got


# ------------------------------------------------------------------ config 1 (paper params)
def test_config1_random_1mib_vs_r1(pkg):
    data = synthgen.random_bytes(1, 1 << 20)
    ch = pkg.Chunker(pkg.Params())
    assert ch.path == "k63"
    got = check_chunk(ch, data, method=1)
    assert got.size == 132
    chb = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536))
    got = check_chunk(chb, data, method=1)
    assert got.size == 102


@pytest.mark.parametrize("n", [0, 1, 2, 47, 48, 49, 50, 97, 255, 4095, 4096, 4097, 70001,
                               (1 << 20) + 13, (5 << 20) + 12345])
def test_lengths_dense_and_default(pkg, n):
    data = synthgen.random_bytes(n + 7, n)
    for p in (pkg.Params(), pkg.Params(divisor=16, magic=8), pkg.Params(divisor=2, magic=1)):
        check_chunk(pkg.Chunker(p), data)


@pytest.mark.parametrize("offset", [1, 3, 7, 8, 13, 15])
def test_unaligned_base(pkg, offset):
    data = synthgen.random_bytes(100 + offset, (3 << 20) + 77)
    check_chunk(pkg.Chunker(pkg.Params(divisor=256)), data, offset)


def test_many_rows_and_ragged_tail(pkg):
    data = synthgen.random_bytes(5, (37 << 20) + 4093)
    for p in (pkg.Params(), pkg.Params(divisor=512, magic=3)):
        check_chunk(pkg.Chunker(p), data)


def test_special_inputs(pkg):
    ch = pkg.Chunker(pkg.Params())
    n = (2 << 20) + 5
    z = np.zeros(n, np.uint8)
    assert check_chunk(ch, z).size == 0
    check_chunk(ch, np.full(n, 0xFF, np.uint8))
    check_chunk(ch, synthgen.text_like(3, n))
    # adversarial: a candidate every 2 bytes -> per-row lists overflow -> exact re-roll
    per = synthgen.periodic(b"\x04\xd5", n)
    got = check_chunk(ch, per)
    assert got.size == (n - 48 + 1) // 2
    chb = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536))
    check_chunk(chb, per)
    check_chunk(chb, z)


def test_k32_path(pkg):
    p = pkg.Params(poly=0x104C11DB7)
    ch = pkg.Chunker(p)
    assert ch.path == "k32"
    for n, seed in (((4 << 20) + 3, 1), (100000, 2)):
        check_chunk(ch, synthgen.random_bytes(seed, n))
    check_chunk(pkg.Chunker(pkg.Params(poly=0x104C11DB7, divisor=64, magic=5)),
                synthgen.random_bytes(9, (3 << 20) + 1))


SMALL_LIMIT = 147 * 1024 * 32       # bulk bytes up to which the small launch shape runs (148 SMs)


@pytest.mark.parametrize("poly", [LBFS, 0x104C11DB7, 0x20000005])   # K63, K32B, K32 (deg 29)
@pytest.mark.parametrize("n", [(4 << 20) + 4093, SMALL_LIMIT + 60, SMALL_LIMIT + 100, (5 << 20) + 1])
def test_launch_shapes_around_small_threshold(pkg, poly, n):
    """Inputs up to ~4.6 MiB run the small launch shape (128 consumers x 2 rows per CTA), larger
    ones the big shape; both sides of the switch, every u32/u64 kernel mode, and a dense divisor
    (a marker every 64 B on average: many hits per row)."""
    data = synthgen.random_bytes(21, n)
    for p in (pkg.Params(poly=poly), pkg.Params(poly=poly, divisor=64, magic=17)):
        check_chunk(pkg.Chunker(p), data)


def test_long_window_variants(pkg):
    """Windows > 64 on the hot kernel (pops from the second TMA tile, 16 ceil(w/16) bytes behind),
    every marker kind and state mode; inputs below 4 KiB take the generic loop."""
    for p in (pkg.Params(window=65), pkg.Params(window=80, divisor=256, magic=7, marker=1),
              pkg.Params(poly=0x11D, window=70, divisor=128, magic=5, marker=1),
              pkg.Params(window=100, divisor=3000, magic=2999, marker=1),
              pkg.Params(window=65, divisor=1 << 40, magic=12345),
              pkg.Params(poly=0x80002001, window=96), pkg.Params(poly=0x104C11DB7, window=129, divisor=512),
              pkg.Params(poly=0x8000000000000801, window=255, divisor=1024, magic=3),
              pkg.Params(window=4096, divisor=256), pkg.Params(window=1000, min_size=512, max_size=4096)):
        ch = pkg.Chunker(p)
        assert ch.path in ("k63", "k32")
        check_chunk(ch, synthgen.random_bytes(11, 300000))
        check_chunk(ch, synthgen.random_bytes(12, (3 << 20) + 77), offset=5)
        check_chunk(ch, synthgen.random_bytes(13, 3000))                       # generic loop
    # the '<=' marker with any window <= 64 runs on the hot kernel (funnel-shifted pops)
    for p in (pkg.Params(window=1, divisor=256, magic=7, marker=1),
              pkg.Params(poly=(1 << 63) | 3, window=24, divisor=1024, marker=1)):
        ch = pkg.Chunker(p)
        assert ch.path == "k63"
        check_chunk(ch, synthgen.random_bytes(11, 300000))


def test_bounded_variants(pkg):
    data = synthgen.random_bytes(12, (6 << 20) + 99)
    for D in (2048, 8192, 65536):
        for mn, mx in ((D // 4, 8 * D), (0, 4 * D), (D, D), (1, 1)):
            check_chunk(pkg.Chunker(pkg.Params(divisor=D, min_size=mn, max_size=mx)), data)


# ------------------------------------------------------------------ split invariance (T3/T5)
@pytest.mark.parametrize("G", [1, 2, 3, 8])
def test_virtual_shards_concatenate_to_chunk(pkg, G):
    n = (9 << 20) + 321
    data = synthgen.random_bytes(13, n)
    ch = pkg.Chunker(pkg.Params(divisor=1024))
    exp = oracle.candidates(data, oracle.Params(divisor=1024))
    parts = []
    bounds = [n * g // G for g in range(G + 1)]
    for g in range(G):
        a, b = bounds[g], bounds[g + 1]
        halo = min(47, a)
        x = dev(data[a - halo:b])
        parts.append(ch.candidates_range(x, halo, a, n).cpu().numpy())
    got = np.concatenate(parts).astype(np.uint64)
    assert np.array_equal(got, exp)
    # the global size-bound pass over the concatenation (bounded mode across shards)
    chb = pkg.Chunker(pkg.Params(divisor=1024, min_size=256, max_size=8192))
    cuts = chb.size_bound(torch.from_numpy(got.astype(np.int64)).cuda(), n).cpu().numpy()
    assert np.array_equal(cuts.astype(np.uint64), oracle.size_bound(exp, n, 256, 8192))


@pytest.mark.parametrize("mn,mx", [(256, 8192), (4096, 65536), (16384, 0)])
def test_size_bound_state_chains_over_virtual_shards(pkg, mn, mx):
    """shred_size_bound_state: chaining the rule over shard ranges through the exit states equals
    the whole-stream rule (the per-rank step of the distributed size rule, f1); min < D (blocks
    of 8), min = 4D (repair passes) and min = 16D (the serial walk), with held cuts at the
    shard ends."""
    n = (9 << 20) + 321
    data = synthgen.random_bytes(17, n)
    p = pkg.Params(divisor=1024, min_size=mn, max_size=mx)
    ch = pkg.Chunker(p)
    cand = oracle.candidates(data, oracle.Params(divisor=1024)).astype(np.int64)
    exp = oracle.size_bound(cand.astype(np.uint64), n, mn, mx)
    for G in (1, 3, 8):
        bounds = [n * g // G for g in range(G + 1)]
        s, held, got = 0, False, []
        for g in range(G):
            a, b = bounds[g], bounds[g + 1]
            part = torch.from_numpy(cand[(cand > a) & (cand <= b)].copy())
            cuts, s, held = ch.size_bound_state(part, b, b == n, s, held)
            got.append(cuts.cpu().numpy())
        assert np.array_equal(np.concatenate(got).astype(np.uint64), exp)


def test_size_bound_state_dev_chains_with_device_states(pkg):
    """shred_size_bound_state_dev: the same chaining with the candidate count and the entry
    state read from device memory and the exit state left there (no host value between the
    pieces); the candidate buffer is larger than the count (the count bounds the work)."""
    n = (7 << 20) + 99
    data = synthgen.random_bytes(18, n)
    p = pkg.Params(divisor=512, min_size=300, max_size=4000)
    ch = pkg.Chunker(p)
    cand = oracle.candidates(data, oracle.Params(divisor=512)).astype(np.int64)
    exp = oracle.size_bound(cand.astype(np.uint64), n, 300, 4000)
    G = 5
    bounds = [n * g // G for g in range(G + 1)]
    state = torch.zeros(2, dtype=torch.int64, device="cuda")
    outs = []
    for g in range(G):
        a, b = bounds[g], bounds[g + 1]
        part = cand[(cand > a) & (cand <= b)]
        buf = torch.full((part.size + 100,), -1, dtype=torch.int64, device="cuda")
        buf[:part.size] = torch.from_numpy(part.copy()).cuda()
        nd = torch.tensor([part.size], dtype=torch.int64, device="cuda")
        out = torch.empty(part.size + (b - a) // 4000 + 8, dtype=torch.int64, device="cuda")
        no = torch.zeros(1, dtype=torch.int64, device="cuda")
        ch.size_bound_state_dev(buf, nd, b, b == n, state, out, no, state)
        outs.append((out, no))
    got = np.concatenate([o[:int(k.item())].cpu().numpy() for o, k in outs]).astype(np.uint64)
    assert np.array_equal(got, exp)


# ------------------------------------------------------------------ streaming (config 3 shape)
def _feed_all(ch, data, sizes, pinned):
    outs = []
    off = 0
    for s in sizes:
        piece = torch.from_numpy(data[off:off + s].copy())
        x = piece.pin_memory() if pinned else piece.cuda()
        outs.append(ch.feed(x).cpu().numpy())
        off += s
    outs.append(ch.flush().cpu().numpy())
    return np.concatenate(outs).astype(np.uint64)


@pytest.mark.parametrize("pinned", [False, True])
@pytest.mark.parametrize("bounded", [False, True])
def test_feed_matches_one_shot(pkg, pinned, bounded):
    n = (3 << 20) + 555
    data = synthgen.random_bytes(14, n)
    p = pkg.Params(divisor=2048, min_size=512 if bounded else 0, max_size=16384 if bounded else 0)
    exp = oracle.chunk(data, oparams(p))
    ch = pkg.Chunker(p)
    ch.set_ring(3, 1 << 20)                       # host pieces larger than a slot get split
    rng = np.random.default_rng(5)
    sizes = []
    left = n
    while left:
        s = int(min(left, rng.choice([1, 2, 47, 48, 1000, 65536, 1 << 20, (1 << 21) + 3])))
        sizes.append(s); left -= s
    got = _feed_all(ch, data, sizes, pinned)
    assert np.array_equal(got, exp)
    # the ctx is reusable for a second stream
    got2 = _feed_all(ch, data, [n // 2, n - n // 2], pinned)
    assert np.array_equal(got2, exp)


@pytest.mark.parametrize("window,poly,marker", [(47, LBFS, 0), (33, 0x104C11DB7, 0), (9, 0x20000005, 0),
                                               (47, LBFS, 1), (31, 0x104C11DB7, 1)])
def test_feed_and_shards_funnel_windows(pkg, window, poly, marker):
    """Windows that are not a multiple of 16 (funnel pops on the hot kernel) through the
    streaming carry (w-1 bytes across feeds, pinned and device pieces) and through byte-range
    shards with a w-1 halo: both equal the oracle on the whole stream."""
    n = (3 << 20) + 4321
    data = synthgen.random_bytes(40 + window, n)
    p = pkg.Params(poly=poly, window=window, divisor=1024, magic=window, marker=marker)
    op = oparams(p)
    exp = oracle.chunk(data, op)
    ch = pkg.Chunker(p)
    assert ch.path in ("k63", "k32")
    ch.set_ring(2, 1 << 20)
    sizes = [1, window - 1, 70000, (1 << 20) + 5, 3, n - (1 + window - 1 + 70000 + (1 << 20) + 5 + 3)]
    assert np.array_equal(_feed_all(ch, data, sizes, pinned=True), exp)
    assert np.array_equal(_feed_all(ch, data, sizes[::-1], pinned=False), exp)
    G = 3
    bounds = [n * g // G for g in range(G + 1)]
    parts = []
    for g in range(G):
        a, b = bounds[g], bounds[g + 1]
        halo = min(window - 1, a)
        parts.append(ch.candidates_range(dev(data[a - halo:b]), halo, a, n).cpu().numpy())
    assert np.array_equal(np.concatenate(parts).astype(np.uint64), oracle.candidates(data, op))
    chb = pkg.Chunker(pkg.Params(poly=poly, window=window, divisor=1024, magic=window,
                                 min_size=256, max_size=8192, marker=marker))
    assert np.array_equal(_feed_all(chb, data, sizes, pinned=True),
                          oracle.chunk(data, oparams(chb.params)))


def test_feed_candidate_at_piece_boundary(pkg):
    """A candidate exactly at a feed end is held, emitted once more data arrives."""
    data = synthgen.periodic(b"\x04\xd5", 4000)
    p = pkg.Params()
    exp = oracle.chunk(data, oracle.Params())
    ch = pkg.Chunker(p)
    got = _feed_all(ch, data, [100, 1, 1, 898, 3000], pinned=False)   # 100, 102 are candidates
    assert np.array_equal(got, exp)


# ------------------------------------------------------------------ device generator
def test_synth_fill_matches_host_generator(pkg):
    for seed, off, n in ((1, 0, 1 << 20), (5, 3, 100003), (7, (1 << 33) + 5, 4099)):
        t = torch.empty(n, dtype=torch.uint8, device="cuda")
        pkg.synth_fill(t, seed, off)
        assert np.array_equal(t.cpu().numpy(), synthgen.random_bytes(seed, n, off))


# ------------------------------------------------------------------ full-size configs
def test_config2_1gib_and_edited_version(pkg):
    """configs[1]: 1 GiB + an edited version, device-resident, in bench.py's launch config.
    Exact vs oracle R2 (multithreaded) on both versions; edit locality on the candidates."""
    n = 1 << 30
    base = torch.empty(n, dtype=torch.uint8, device="cuda")
    pkg.synth_fill(base, 2)
    ch = pkg.Chunker(pkg.Params())
    got = ch.chunk(base).cpu().numpy().astype(np.uint64)
    host = base.cpu().numpy()
    assert np.array_equal(host[:4096], synthgen.random_bytes(2, 4096))
    exp = oracle.candidates(host)
    assert np.array_equal(got, exp)
    mu = (n - 48) / 8192
    assert abs(got.size - mu) < 5 * np.sqrt(mu)
    ed, ops = synthgen.edited(host, 3)
    got2 = ch.chunk(dev(ed)).cpu().numpy().astype(np.uint64)
    assert np.array_equal(got2, oracle.candidates(ed))
    # bounded mode on the base (sampled: every cut verified by the size-rule characterisation)
    chb = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536))
    cuts = chb.chunk(base).cpu().numpy().astype(np.uint64)
    assert np.array_equal(cuts, oracle.size_bound(exp, n, 2048, 65536))


# ------------------------------------------------------------------ size rule (a5) in isolation
def _sb_cases():
    rng = np.random.default_rng(17)
    yield np.arange(48, 200000, 2, dtype=np.uint64), 200001, 3, 0          # phases never sync
    yield np.arange(48, 200000, 2, dtype=np.uint64), 200001, 5, 9
    yield np.arange(48, 300000, 3, dtype=np.uint64), 300000, 4, 0
    yield np.zeros(0, np.uint64), 1 << 20, 2048, 65536                    # forced cuts only
    yield np.array([5], np.uint64), 10, 0, 3
    yield np.unique(rng.integers(1, 1 << 26, 200000)).astype(np.uint64), 1 << 26, 256, 1024
    yield np.unique(rng.integers(1, 1 << 30, 5000)).astype(np.uint64), 1 << 30, 2048, 65536  # long gaps
    c = np.unique(rng.integers(1, 1 << 22, 100000)).astype(np.uint64)
    yield c, 1 << 22, 0, 64
    yield c, 1 << 22, 64, 64
    yield c, 1 << 22, 1, 1


def test_size_bound_api_vs_oracle(pkg):
    for cand, n, mn, mx in _sb_cases():
        ch = pkg.Chunker(pkg.Params(divisor=2, magic=0, min_size=mn, max_size=mx))
        got = ch.size_bound(torch.from_numpy(cand.astype(np.int64)).cuda(), n).cpu().numpy()
        exp = oracle.size_bound(cand, n, mn, mx)
        assert np.array_equal(got.astype(np.uint64), exp), (len(cand), n, mn, mx)


def test_bounded_adversarial_stream(pkg):
    """(04 D5)* gives a candidate every 2 bytes: with min = 3 the blocks' speculative runs are
    out of phase half the time, so the exact sequential fallback of sb_plan is exercised."""
    n = (4 << 20) + 11
    per = synthgen.periodic(b"\x04\xd5", n)
    for mn, mx in ((3, 0), (3, 1000), (4097, 65536)):
        check_chunk(pkg.Chunker(pkg.Params(min_size=mn, max_size=mx)), per)


# ------------------------------------------------------------------ variants (f4)
def test_marker_le_and_non_pow2_divisor(pkg):
    """Divisors that are not powers of two (Q8: the integer remainder of the fingerprint's value):
    the '==' marker runs on the hot kernel (divisibility test on the full state), the
    "value mod p <= constant" set (L249-L251) too (the remainder by a multiply-high quotient);
    bit-exact vs the oracle, bounded mode on top."""
    data = synthgen.random_bytes(31, (2 << 20) + 77)
    for p, path in ((pkg.Params(divisor=10000, magic=1234), "k63"),
                    (pkg.Params(divisor=12345, magic=3, marker=1), "k63"),
                    (pkg.Params(divisor=3, magic=0), "k63"),
                    (pkg.Params(divisor=3000, magic=2999, min_size=1000, max_size=20000), "k63"),
                    (pkg.Params(divisor=5000, magic=4, marker=1, min_size=1000, max_size=20000), "k63")):
        ch = pkg.Chunker(p)
        assert ch.path == path
        check_chunk(ch, data)


@pytest.mark.parametrize("bounded", [False, True])
def test_le_marker_dense_rate_lists_sized_by_rate(pkg, bounded):
    """'<=' marker with r near D (hit rate (r+1)/D up to 1/2): the per-row lists are sized by the
    set's rate, so bounded mode stays on the parallel size-rule kernels instead of
    the one-CTA dense walk; exact vs the oracle either way (L249-L251)."""
    data = synthgen.random_bytes(41, (6 << 20) + 333)
    for D, r in ((8192, 4095), (8192, 511), (256, 127)):
        p = pkg.Params(divisor=D, magic=r, marker=1, min_size=64 if bounded else 0,
                       max_size=4096 if bounded else 0)
        check_chunk(pkg.Chunker(p), data)


def test_two_streams_one_ctx_are_ordered(pkg):
    """Two one-shot calls on two different streams of one ctx (shared scratch and aux) give the
    same results as on one stream: the library orders them."""
    a = synthgen.random_bytes(51, (32 << 20) + 5)
    b = synthgen.random_bytes(52, (3 << 20) + 7)
    ch = pkg.Chunker(pkg.Params())
    xa, xb = dev(a), dev(b)
    oa = torch.empty(1 << 16, dtype=torch.int64, device="cuda")
    ob = torch.empty(1 << 16, dtype=torch.int64, device="cuda")
    na = torch.zeros(1, dtype=torch.int64, device="cuda")
    nb = torch.zeros(1, dtype=torch.int64, device="cuda")
    s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()
    torch.cuda.synchronize()
    for _ in range(5):
        ch.chunk_async(xa, oa, na, stream=s1)
        ch.chunk_async(xb, ob, nb, stream=s2)
    torch.cuda.synchronize()
    ea, eb = oracle.candidates(a), oracle.candidates(b)
    assert int(na.item()) == ea.size and int(nb.item()) == eb.size
    assert np.array_equal(oa[:ea.size].cpu().numpy().astype(np.uint64), ea)
    assert np.array_equal(ob[:eb.size].cpu().numpy().astype(np.uint64), eb)


@pytest.mark.parametrize("poly", [LBFS, 0x104C11DB7, 0x20000005, None])   # K63, K32B, K32, K40
@pytest.mark.parametrize("D", [3, 7, 10000, 3 << 20, 3 << 31, (1 << 40) + 1, 12345678901, (1 << 32) - 1])
def test_non_pow2_divisor_hot_kernel(pkg, poly, D):
    """'==' marker with D = d 2^s (d odd > 1, s < 32) on the hot kernel: f mod D == r iff
    rotr64((f + D - r) d^-1, s) <= floor((2^64-1)/D).  Large D hit nothing on random data, so r is
    planted from real window fingerprints (oracle R2); a funnel window (w = 47) and a feed too."""
    if poly is None:
        poly = _dense_irreducible(37, 37)
    k = oracle.degree(poly)
    if D > (1 << k):
        pytest.skip("D <= 2^deg")
    data = synthgen.random_bytes(int(D % 1000) + k, (3 << 20) + 333)
    fps = oracle.window_fps(data, oracle.Params(poly=poly))
    for w, r in ((48, int(fps[fps.size // 3]) % D), (47, 1 % D)):
        p = pkg.Params(poly=poly, window=w, divisor=D, magic=r)
        ch = pkg.Chunker(p)
        assert ch.path == ("k63" if k >= 33 else "k32")
        got = check_chunk(ch, data, offset=w % 16)
        if w == 48:
            assert got.size >= 1
    # streaming with the carry across pinned pieces
    ch = pkg.Chunker(pkg.Params(poly=poly, divisor=D, magic=int(fps[7]) % D))
    exp = oracle.chunk(data, oparams(ch.params))
    n = data.size
    assert np.array_equal(_feed_all(ch, data, [n // 3, 47, n - n // 3 - 47], True), exp)


@pytest.mark.parametrize("poly,path", [(LBFS, "k63"), (0x104C11DB7, "k32")])
@pytest.mark.parametrize("window", [16, 32, 48, 64])
@pytest.mark.parametrize("marker", [0, 1])
def test_fast_path_windows_and_le_marker(pkg, poly, path, window, marker):
    """The hot kernel's instances: w in {16,32,48,64} x {==, <=} marker sets, both degrees."""
    D, r = (4096, 9) if marker else (1024, 77)
    p = pkg.Params(poly=poly, window=window, divisor=D, magic=r, marker=marker)
    ch = pkg.Chunker(p)
    assert ch.path == path
    check_chunk(ch, synthgen.random_bytes(window + marker, (3 << 20) + 31), offset=5)


@pytest.mark.parametrize("poly", [LBFS, 0x104C11DB7, 0x20000005, None])   # K63, K32B, K32, K40
@pytest.mark.parametrize("window", [1, 2, 7, 15, 17, 31, 33, 47, 49, 63])
def test_fast_path_any_window(pkg, poly, window):
    """Windows that are not a multiple of 16 on the hot kernel: the bytes leaving the window are a
    funnel (PRMT) of two staged 16-byte chunks at offset e = 16 ceil(w/16) - w; every state mode."""
    if poly is None:
        poly = _dense_irreducible(37, 37)
    p = pkg.Params(poly=poly, window=window, divisor=512, magic=window % 512)
    ch = pkg.Chunker(p)
    assert ch.path in ("k63", "k32")
    data = synthgen.random_bytes(100 + window, (2 << 20) + 4 * window + 1)
    check_chunk(ch, data, offset=window % 16)
    # the '<=' marker set (L249-L251) with the same funnel windows
    chl = pkg.Chunker(pkg.Params(poly=poly, window=window, divisor=512, magic=3, marker=1))
    assert chl.path == ch.path
    check_chunk(chl, data, offset=(window + 3) % 16)


def _dense_irreducible(deg, seed):
    rng = np.random.default_rng(seed)
    while True:
        low = int(rng.integers(0, 1 << min(deg, 62))) | 1
        p = (1 << deg) | (low & ((1 << deg) - 1))
        if oracle.is_irreducible(p):
            return p


@pytest.mark.parametrize("deg", [8, 9, 12, 16, 24, 31, 32, 33, 40, 41, 48, 57, 62, 63])
def test_polynomial_degrees(pkg, deg):
    """Any degree: u32-state fast kernel for 8..32 (8, 16, 24, 32: the top byte is a whole byte,
    PRMT index), u64-state for 33..63 (top byte by mulhi for 41..63, by a funnel shift for
    33..40); T tables with the (t << k) cancel term; dense random irreducible P, bit-exact."""
    P = _dense_irreducible(deg, deg)
    D = 1 << min(10, deg - 1)
    p = pkg.Params(poly=P, divisor=D, magic=D // 3)
    ch = pkg.Chunker(p)
    assert ch.path == ("k32" if deg <= 32 else "k63")
    check_chunk(ch, synthgen.random_bytes(deg, (2 << 20) + 123), offset=deg % 16)


@pytest.mark.parametrize("poly", [LBFS, 0x104C11DB7])
@pytest.mark.parametrize("log2d", [1, 20, 31, 32, 33])
def test_divisor_range_with_planted_magic(pkg, poly, log2d):
    """D from 2 up to past the hot kernel's 2^32 limit (the marker test keeps the low log2 D
    bits at the top of a u32: D = 2^32 is the shift-by-0 edge).  On random data a large D hits
    nothing, so r is planted: the residue of three real window fingerprints (oracle R2), and the
    candidate set must be exactly the positions sharing it."""
    if poly != LBFS and log2d > 32:
        pytest.skip("deg 32: D <= 2^32")
    data = synthgen.random_bytes(700 + log2d, (3 << 20) + 77)
    op = oracle.Params(poly=poly)
    fps = oracle.window_fps(data, op)
    D = 1 << log2d
    for k in (5, fps.size // 2, fps.size - 9):
        r = int(fps[k]) % D
        p = pkg.Params(poly=poly, divisor=D, magic=r)
        ch = pkg.Chunker(p)
        assert ch.path == ("k63" if poly == LBFS else "k32")
        got = check_chunk(ch, data)
        if log2d >= 20:
            exp = np.nonzero((fps % np.uint64(D)) == np.uint64(r))[0].astype(np.uint64) + np.uint64(op.window)
            exp = exp[exp < data.size]
            assert np.array_equal(got, exp) and got.size >= 1


@pytest.mark.parametrize("window", [1, 7, 16, 47, 48, 64])
@pytest.mark.parametrize("marker", [0, 1])
def test_degree8_fast_path(pkg, window, marker):
    """deg P = 8: the whole state is the top byte, so the u32 kernel's PRMT byte index applies
    (f <- ((f << 8) | b) ^ T[f] ^ U[o], T carrying the t << 8 cancel term); D <= 2^8.  Sizes on
    both launch shapes (1 MiB: small; 6 MiB: big), an unaligned base, and the streaming carry."""
    P = 0x11D
    for D, r in ((256, 0x78 if not marker else 9), (64, 5), (2, 1 if not marker else 0)):
        p = pkg.Params(poly=P, window=window, divisor=D, magic=r, marker=marker)
        ch = pkg.Chunker(p)
        assert ch.path == "k32"
        data = synthgen.random_bytes(800 + window + D, (1 << 20) + 77 if D != 256 else (6 << 20) + 5)
        check_chunk(ch, data, offset=window % 16)
    ch = pkg.Chunker(pkg.Params(poly=P, window=window, divisor=256, magic=3, marker=marker))
    data = synthgen.random_bytes(900 + window, (2 << 20) + 11)
    n = data.size
    assert np.array_equal(_feed_all(ch, data, [n // 2, 1, n - n // 2 - 1], True), oracle.chunk(data, oparams(ch.params)))


@pytest.mark.parametrize("poly", [LBFS, 0x104C11DB7, 0x20000005, None, 0x11D])   # K63, K32B, K32, K40, deg 8
@pytest.mark.parametrize("D", [3, 255, 10000, 3 << 20, (1 << 32) - 1, 1 << 33, 3 << 32, (1 << 40) + 1,
                               12345678901, (1 << 62) + 12345, 1 << 63])
def test_remainder_marker_hot_kernel(pkg, poly, D):
    """MK_REM: the '<=' set (L249-L251) with any D, and '==' where 2^32 | D, on the hot kernel:
    rem = f - q D with q = mulhi64(f, ceil(2^(63+l) / D)) >> (l-1), l = ceil(log2 D) (exact for
    f < 2^63).  r is planted from real window fingerprints (oracle R2): for '<=' the smallest
    residue of the first 4096 windows (about one hit per 4096 B), for '==' one residue; a funnel
    window (w = 47) and a streaming feed too."""
    if poly is None:
        poly = (1 << 40) | 0x39
    deg = poly.bit_length() - 1
    if not oracle.is_irreducible(poly):
        pytest.skip("not irreducible")
    if D > (1 << deg):
        pytest.skip("D > 2^deg")
    data = synthgen.random_bytes(900 + (D % 97), (3 << 20) + 41)
    for w in (48, 47):
        op = oracle.Params(poly=poly, window=w)
        fps = oracle.window_fps(data, op)
        res = fps[:4096] % np.uint64(D)
        cases = [(1, int(res.min()))]
        if D % (1 << 32) == 0 or (D & (D - 1)) != 0:
            cases.append((0, int(fps[fps.size // 3]) % D))
        for marker, r in cases:
            p = pkg.Params(poly=poly, window=w, divisor=D, magic=r, marker=marker)
            ch = pkg.Chunker(p)
            assert ch.path == ("k63" if deg >= 33 else "k32")
            got = check_chunk(ch, data, offset=w % 16)
            hit = (fps % np.uint64(D)) <= np.uint64(r) if marker else (fps % np.uint64(D)) == np.uint64(r)
            exp = np.nonzero(hit)[0].astype(np.uint64) + np.uint64(w)
            assert np.array_equal(got, exp[exp < data.size]) and got.size >= 1
    ch = pkg.Chunker(pkg.Params(poly=poly, window=47, divisor=D, magic=r, marker=marker))
    n = data.size
    assert np.array_equal(_feed_all(ch, data, [n // 3, 5, n - n // 3 - 5], True), oracle.chunk(data, oparams(ch.params)))


# ------------------------------------------------------------------ K32T (T as an integer product)
@pytest.mark.parametrize("poly", [0x80002001, 0x80040001, 0x40200001, 0x10000201, 0x800201, 0x40201,
                                  0x8000000000000801])     # the last: K63T (u64 state)
@pytest.mark.parametrize("window,marker", [(48, 0), (48, 1), (32, 0), (47, 0), (16, 1)])
def test_k32t_multiply_reduction_paths(pkg, poly, window, marker):
    """Sparse irreducible P (Q's terms >= 8 apart): the u32 kernel reduces the top byte with one
    IMAD (MODE_K32T, L255-L258 with any irreducible div(x)); bit-exact vs the oracle with both
    marker sets, funnel windows, bounds, a feed straddling pieces, and virtual shards."""
    data = synthgen.random_bytes(poly & 0xFFFF, (3 << 20) + 4093)
    D = 512 if poly < (1 << 20) else 4096
    p = pkg.Params(poly=poly, window=window, divisor=D, magic=7 if not marker else 3, marker=marker)
    ch = pkg.Chunker(p)
    assert (ch.mode, ch.path) == (("k63t", "k63") if poly >> 40 else ("k32t", "k32"))
    got = check_chunk(ch, data)
    pb = pkg.Params(poly=poly, window=window, divisor=D, magic=7 if not marker else 3, marker=marker,
                    min_size=D // 4, max_size=8 * D)
    check_chunk(pkg.Chunker(pb), data)
    # feed in uneven pieces (carry across pieces), then two virtual shards
    chf = pkg.Chunker(p)
    outs, a = [], 0
    for step in (1 << 20, 12345, (1 << 21) + 1, len(data)):
        outs.append(chf.feed(dev(data[a:a + step])).cpu().numpy())
        a = min(len(data), a + step)
    outs.append(chf.flush().cpu().numpy())
    assert np.array_equal(np.concatenate(outs).astype(np.uint64), got)
    n = len(data)
    s = (n // 2) // 4096 * 4096
    x = dev(data)
    parts = [ch.candidates_range(x[:s], 0, 0, n), ch.candidates_range(x[s - (window - 1):], window - 1, s, n)]
    assert np.array_equal(torch.cat(parts).cpu().numpy().astype(np.uint64), oracle.candidates(data, oparams(p)))


def test_k32t_small_shape_and_le_marker_modes(pkg):
    """1 MiB (the small launch shape) on K32T; '==' with 2^32 > D; mode selection table."""
    data = synthgen.random_bytes(77, 1 << 20)
    for p, mode in ((pkg.Params(poly=0x80002001), "k32t"),
                    (pkg.Params(poly=0x80002001, divisor=1 << 20, magic=12345), "k32t"),
                    (pkg.Params(poly=0x80002001, divisor=10000, magic=7), "k32"),      # MK_DIV: table mode
                    (pkg.Params(poly=0x104C11DB7), "k32b"), (pkg.Params(), "k63"),
                    (pkg.Params(poly=0x8000000000000801), "k63t"),
                    (pkg.Params(poly=0x8000000000000801, divisor=10000, magic=9), "k63")):
        ch = pkg.Chunker(p)
        assert ch.mode == mode, (p, ch.mode)
        check_chunk(ch, data)


# ------------------------------------------------------------------ one-CTA size rule (sb_one)
def _periodic_marker_pattern(period: int, p) -> bytes:
    """A random `period`-byte pattern one of whose window phases is a marker under p (found with
    the oracle), so its repetition has a candidate every `period` bytes."""
    rng = np.random.default_rng(period)
    for _ in range(200000):
        pat = bytes(rng.integers(0, 256, period, dtype=np.uint8))
        if oracle.candidates(synthgen.periodic(pat, 3 * period + p.window), oparams(p)).size:
            return pat
    raise AssertionError("no marker pattern found")


@pytest.mark.parametrize("kind", ["random", "periodic64", "dense04d5", "short"])
def test_bounded_one_shot_one_cta_paths(pkg, kind):
    """One-shot bounded calls with few expected candidates run the whole size rule in one CTA
    (sb_one): its shared-memory form (random data), its global-memory phases (> 8,176 actual
    candidates without list overflow: a 64-byte period with a marker, 16 K candidates per MiB),
    and its dense form (list overflow, `04 D5`); all equal the oracle (L259-L265)."""
    p = pkg.Params(min_size=16, max_size=200) if kind != "random" else pkg.Params(min_size=2048, max_size=65536)
    n = (1 << 20) + 13
    if kind == "random":
        data = synthgen.random_bytes(77, n)
    elif kind == "periodic64":
        data = synthgen.periodic(_periodic_marker_pattern(64, pkg.Params()), n)
    elif kind == "dense04d5":
        data = synthgen.periodic(b"\x04\xd5", n)
    else:
        data = synthgen.random_bytes(78, 1000)
    got = check_chunk(pkg.Chunker(p), data)
    if kind == "periodic64":
        assert oracle.candidates(data, oparams(p)).size > 8176
    if kind != "short":
        assert got.size > 0


@pytest.mark.parametrize("mn,mx", [(8192, 65536), (65536, 0), (131072, 262144), (40000, 40001)])
def test_bounded_min_above_d_serial_walk(pkg, mn, mx):
    """min >= D: blocks of 16 candidates often fail to re-sync with their speculation, so the size
    rule runs its repair passes (super-blocks of 1 and 32 blocks) and, when they do not converge
    (min >~ 16D), its ballot walk; equal to the oracle (L259-L265) on 80 MiB of random data, with
    and without forced cuts, and on 6 MiB (the one-CTA form)."""
    data = synthgen.random_bytes(91, (80 << 20) + 333)       # > 8,192 expected candidates: the multi-CTA rule
    ch = pkg.Chunker(pkg.Params(min_size=mn, max_size=mx))
    check_chunk(ch, data)
    check_chunk(ch, data[: (6 << 20) + 5])                  # few candidates: sb_one (shared-memory form)

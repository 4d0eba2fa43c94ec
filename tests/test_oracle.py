"""Pins for the CPU oracle (tier T0/T1/T4 of SURVEY.md §4.2) — no GPU needed.

Each test pins the oracle to something other than itself: CRC catalogue values, closed forms,
Gauss's count of irreducible polynomials, Python big-integer brute force, invariants the paper
states (split independence L282-L287, edit locality L1150-L1153) and exact statistics.
"""
import os

import numpy as np
import pytest

import oracle
from oracle import Params, brute
import synthgen

LBFS = oracle.LBFS_POLY


def _golden(golden_dir, name):
    rows = []
    with open(os.path.join(golden_dir, name)) as f:
        for line in f:
            line = line.strip()
            if line and not line.startswith("#"):
                rows.append(line.split())
    return rows


# --------------------------------------------------------------------------- reducer / bit order
def test_crc_catalogue_pins_reducer_and_bit_order(golden_dir):
    """R1(M || 0^{width/8}) == CRC(M) XOR xorout for init-0 non-reflected CRCs (Q4)."""
    rows = _golden(golden_dir, "crc_catalogue.txt")
    assert len(rows) >= 5
    for name, width, poly, xorout, check in rows:
        width, poly, xorout, check = int(width), int(poly, 16), int(xorout, 16), int(check, 16)
        msg = b"123456789" + b"\0" * (width // 8)
        if width == 64:
            got = oracle.polymod(msg, poly, deg=64)
        else:
            got = oracle.polymod(msg, (1 << width) | poly)
        assert got ^ xorout == check, name


def test_brute_force_matches_catalogue_too(golden_dir):
    """The Python brute force is pinned by the same catalogue (so it can pin R1)."""
    for name, width, poly, xorout, check in _golden(golden_dir, "crc_catalogue.txt"):
        width, poly = int(width), int(poly, 16)
        got = brute.window_fp(b"123456789" + b"\0" * (width // 8), (1 << width) | poly)
        assert got ^ int(xorout, 16) == int(check, 16), name


def test_no_reduction_closed_form():
    """Degree < 63 windows are their own remainder: fp = newest bytes as a big-endian int."""
    rng = np.random.default_rng(7)
    for k in range(0, 8):
        tail = rng.integers(0, 256, k, dtype=np.uint8).tobytes()
        win = b"\0" * (48 - k) + tail
        expect = int.from_bytes(tail, "big") if k else 0
        assert oracle.window_fp(np.frombuffer(win, np.uint8), 47) == expect
    win = b"\0" * 41 + bytes(range(1, 8))
    assert oracle.window_fp(np.frombuffer(win, np.uint8), 47) == 0x01020304050607


def test_x63_mod_p_closed_form():
    """x^63 mod P = P - x^63 for deg(P) = 63 (message 0x80 followed by 7 zero bytes)."""
    assert oracle.polymod(b"\x80" + b"\0" * 7, LBFS) == LBFS ^ (1 << 63)
    assert oracle.polymod(b"\x80" + b"\0" * 7, (1 << 63) | 3) == 3


def test_r1_vs_bigint_brute_force_random_windows():
    rng = np.random.default_rng(11)
    polys = [LBFS, 0x104C11DB7, (1 << 63) | 3, 0x11D, 0x11B, (1 << 40) | 0x1234567]
    for p in polys:
        for w in (1, 2, 7, 8, 9, 16, 48, 64):
            for _ in range(20):
                win = rng.integers(0, 256, w, dtype=np.uint8)
                assert oracle.polymod(win, p) == brute.window_fp(win.tobytes(), p), (hex(p), w)


# --------------------------------------------------------------------------- irreducibility
def test_irreducibility_test_matches_gauss_counts(golden_dir):
    for d, count in _golden(golden_dir, "irreducible_counts.txt"):
        d, count = int(d), int(count)
        n = sum(oracle.is_irreducible((1 << d) | low) for low in range(1 << d))
        assert n == count, d


def test_paper_polynomial_is_irreducible():
    """div(x) must be irreducible (L255-L256): the LBFS P (reading Q1) and the k=32 variant."""
    assert oracle.is_irreducible(LBFS)
    assert oracle.degree(LBFS) == 63
    assert oracle.is_irreducible(0x104C11DB7)
    assert oracle.is_irreducible((1 << 63) | 3)
    assert not oracle.is_irreducible((1 << 63) | 1)          # x^63 + 1 = (x+1)(...)
    def clmul(a, b):
        r = 0
        while b:
            if b & 1:
                r ^= a
            a, b = a << 1, b >> 1
        return r
    # products of two irreducibles are reducible
    assert not oracle.is_irreducible(clmul(0x104C11DB7, (1 << 31) | 0b1001))
    assert not oracle.is_irreducible(clmul(0x11D, 0x11B) )


# --------------------------------------------------------------------------- R2 vs R1, linearity
def test_r2_equals_r1_on_a_million_windows():
    data = synthgen.random_bytes(21, (1 << 20) + 47)
    for p in (Params(), Params(poly=0x104C11DB7)):
        a = oracle.window_fps(data, p, method=1)
        b = oracle.window_fps(data, p, method=2)
        assert a.size >= 1 << 20
        assert np.array_equal(a, b)


def test_r2_tables_are_positional_r1_values():
    C = oracle.r2_tables(Params())
    rng = np.random.default_rng(3)
    for _ in range(200):
        j, b = int(rng.integers(0, 48)), int(rng.integers(0, 256))
        assert int(C[j, b]) == brute.window_fp(bytes([b]) + b"\0" * j, LBFS)


def test_linearity():
    rng = np.random.default_rng(5)
    for _ in range(200):
        a = rng.integers(0, 256, 48, dtype=np.uint8)
        b = rng.integers(0, 256, 48, dtype=np.uint8)
        assert oracle.polymod(a ^ b, LBFS) == oracle.polymod(a, LBFS) ^ oracle.polymod(b, LBFS)


def test_zeros_give_no_candidates():
    z = np.zeros(1 << 16, np.uint8)
    assert np.all(oracle.window_fps(z) == 0)
    assert oracle.candidates(z).size == 0


# --------------------------------------------------------------------------- candidates
@pytest.mark.parametrize("D,r,w,poly", [(2, 1, 48, LBFS), (16, 8, 48, LBFS), (256, 0x78, 48, LBFS),
                                       (8192, 0x78, 48, LBFS), (64, 3, 16, 0x104C11DB7),
                                       (4, 0, 1, 0x11D), (32, 5, 7, (1 << 63) | 3)])
def test_candidates_vs_brute_force(D, r, w, poly):
    data = synthgen.random_bytes(D + w, 3000)
    expect = brute.candidates(data.tobytes(), poly, w, D, r)
    p = Params(poly=poly, window=w, divisor=D, magic=r)
    for method in (1, 2):
        for threads in (1, 3):
            got = oracle.candidates(data, p, method=method, threads=threads)
            assert got.tolist() == expect


def test_edge_lengths():
    p = Params(divisor=2, magic=0)
    for n in (0, 1, 47, 48, 49, 50, 97):
        data = synthgen.random_bytes(9, n)
        got = oracle.candidates(data, p).tolist()
        assert got == brute.candidates(data.tobytes(), LBFS, 48, 2, 0)
        assert all(48 <= c < n for c in got)


def test_periodic_pattern_dense_candidates():
    data = synthgen.periodic(b"\x04\xd5", 600)
    got = oracle.candidates(data).tolist()
    assert got == brute.candidates(data.tobytes(), LBFS, 48, 8192, 0x78)
    assert got == list(range(48, 600, 2))  # survey App. A regression pin, confirmed by brute force


def test_candidate_count_statistics():
    """Random bytes => every full window's fp is uniform on GF(2)^63 => E[#] = (N-w)/D."""
    n = 2 << 20
    data = synthgen.random_bytes(31, n)
    for D in (256, 1024, 8192):
        k = oracle.candidates(data, Params(divisor=D)).size
        mu = (n - 48) / D
        assert abs(k - mu) <= 4 * np.sqrt(mu), (D, k, mu)


def test_split_independence_of_oracle_threads():
    data = synthgen.random_bytes(41, 1 << 20)
    a = oracle.candidates(data, Params(divisor=256), threads=1)
    for t in (2, 5, 8):
        assert np.array_equal(a, oracle.candidates(data, Params(divisor=256), threads=t))


def test_edit_locality_overwrite():
    """Overwriting byte e changes only candidates in [e+1, e+w] (window-local, L1150-L1153)."""
    base = synthgen.random_bytes(51, 4096)
    p = Params(divisor=16, magic=8)
    c0 = set(oracle.candidates(base, p).tolist())
    rng = np.random.default_rng(1)
    nonempty = 0
    for _ in range(100):
        e = int(rng.integers(0, base.size))
        mod = base.copy()
        mod[e] ^= np.uint8(1 + int(rng.integers(0, 255)))
        c1 = set(oracle.candidates(mod, p).tolist())
        diff = c0 ^ c1
        nonempty += bool(diff)
        assert all(e + 1 <= c <= e + 48 for c in diff)
    assert nonempty > 50


def test_edit_locality_insert_delete():
    base = synthgen.random_bytes(61, 1 << 20)
    p = Params(divisor=256)
    c0 = oracle.candidates(base, p)
    for e, L in ((1000, 10), (500000, 4096), (77777, 1)):
        ins = np.concatenate([base[:e], synthgen.random_bytes(99, L), base[e:]])
        c1 = oracle.candidates(ins, p)
        assert np.array_equal(c0[c0 <= e], c1[c1 <= e])
        assert np.array_equal(c0[c0 >= e + 48] + L, c1[c1 >= e + L + 48])
        dele = np.concatenate([base[:e], base[e + L:]])
        c2 = oracle.candidates(dele, p)
        assert np.array_equal(c0[c0 <= e], c2[c2 <= e])
        assert np.array_equal(c0[c0 >= e + L + 48] - L, c2[c2 >= e + 48])


# --------------------------------------------------------------------------- size rule
def check_size_rule(cuts, cands, n, mn, mx):
    """Declarative characterisation of the rule (readings Q13/Q14): from the last cut s, the
    next cut is the first candidate >= max(s+min, s+1) if it lies within s+max, else the forced
    cut s+max;
    after the final cut no candidate >= s+min remains and the tail is <= max."""
    cands = np.asarray(cands, dtype=np.int64)
    s = 0
    for cut in list(cuts) + [None]:
        k = np.searchsorted(cands, s + max(mn, 1), side="left")   # strictly after the last cut
        nxt = int(cands[k]) if k < cands.size else None
        if cut is None:
            assert nxt is None or (mx and nxt - s > mx and s + mx >= n)
            assert not mx or n - s <= mx
            break
        if nxt is not None and (not mx or nxt - s <= mx):
            assert cut == nxt
        else:
            assert mx and cut == s + mx
        assert 0 < cut < n
        s = cut


def test_size_rule_characterisation_random_lists():
    rng = np.random.default_rng(77)
    for trial in range(400):
        n = int(rng.integers(1, 400))
        k = int(rng.integers(0, min(n, 60)))
        cands = np.unique(rng.integers(1, max(2, n), k)) if n > 1 else np.zeros(0, np.int64)
        cands = cands[(cands > 0) & (cands < n)]
        mn = int(rng.integers(0, 40))
        mx = int(rng.choice([0, max(1, mn), mn + int(rng.integers(1, 80))]))
        cuts = oracle.size_bound(cands.astype(np.uint64), n, mn, mx).tolist()
        check_size_rule(cuts, cands, n, mn, mx)


def test_size_rule_off_is_identity():
    c = np.array([5, 9, 100], np.uint64)
    assert oracle.size_bound(c, 200, 0, 0).tolist() == [5, 9, 100]


def test_size_rule_on_random_stream_and_bounded_mean():
    """Bounded mean chunk ~= min + D(1 - e^{-(max-min)/D}) on random data."""
    n = 4 << 20
    data = synthgen.random_bytes(71, n)
    D, mn, mx = 256, 64, 2048
    p = Params(divisor=D, min_size=mn, max_size=mx)
    cand = oracle.candidates(data, p)
    cuts = oracle.chunk(data, p)
    check_size_rule(cuts.tolist(), cand, n, mn, mx)
    lens = np.diff(np.concatenate([[0], cuts.astype(np.int64)]))
    assert lens.min() >= mn and lens.max() <= mx
    expect = mn + D * (1 - np.exp(-(mx - mn) / D))
    assert abs(lens.mean() - expect) / expect < 0.03


# --------------------------------------------------------------------------- survey regression pins
def test_survey_appendix_a_regression_pins(golden_dir):
    rows = _golden(golden_dir, "survey_appendix_a.txt")
    vals = {}
    for row in rows:
        if row[0] == "fp":
            spec, fp = row[1:-1], int(row[-1], 16)
            win = b""
            for tok in spec:
                if tok == "+":
                    continue
                if "x" in tok:
                    cnt, byte = tok.split("x")
                    win += bytes([int(byte, 16)]) * int(cnt)
                else:
                    win += bytes.fromhex(tok)
            assert len(win) == 48
            assert oracle.polymod(win, LBFS) == fp == brute.window_fp(win, LBFS)
        else:
            vals[row[0]] = row[1:]
    data = synthgen.random_bytes(1, 1 << 20)
    assert data[:16].tobytes().hex() == vals["stream_head"][0]
    assert oracle.window_fp(data, 47) == int(vals["fp_at_47"][0], 16)
    c = oracle.candidates(data)
    assert c.size == int(vals["n_candidates"][0])
    assert c[:6].tolist() == [int(x) for x in vals["first"]]
    assert c[-2:].tolist() == [int(x) for x in vals["last"]]
    assert np.array_equal(c, oracle.candidates(data, method=1))
    assert oracle.chunk(data, Params(min_size=2048, max_size=65536)).size == int(vals["n_bounded_2048_65536"][0])


def test_synthgen_splitmix_vector(golden_dir):
    rows = _golden(golden_dir, "splitmix64.txt")
    seed = int(rows[0][1])
    expect = [int(r[0]) for r in rows[1:]]
    assert [int(x) for x in synthgen.splitmix_words(seed, 0, 5)] == expect
    # byte addressing: any (offset, length) window equals the slice of the full stream
    full = synthgen.random_bytes(3, 1000)
    for off, ln in ((0, 1), (1, 7), (13, 100), (999, 1), (8, 8)):
        assert np.array_equal(synthgen.random_bytes(3, ln, off), full[off:off + ln])


# --------------------------------------------------------------------------- variants (f4)
@pytest.mark.parametrize("D,r,marker", [(1000, 7, 0), (3, 0, 0), (12345, 999, 1), (256, 3, 1), (7, 6, 1)])
def test_variant_markers_vs_brute_force(D, r, marker):
    """Non-power-of-two D and the "mod p <= constant" marker set."""
    data = synthgen.random_bytes(D + r, 2500)
    exp = brute.candidates(data.tobytes(), LBFS, 48, D, r, marker)
    p = Params(divisor=D, magic=r, marker=marker)
    for method in (1, 2):
        assert oracle.candidates(data, p, method=method, threads=2).tolist() == exp


def test_le_marker_density():
    """fp mod D <= r on random bytes: density exactly (r+1)/D (fp uniform on GF(2)^63, D | 2^63
    for powers of two; for other D the bias is < D/2^63)."""
    n = 2 << 20
    data = synthgen.random_bytes(33, n)
    for D, r in ((8192, 1), (10000, 4)):
        k = oracle.candidates(data, Params(divisor=D, magic=r, marker=1)).size
        mu = (n - 48) * (r + 1) / D
        assert abs(k - mu) <= 4 * np.sqrt(mu)


# --------------------------------------------------------------------------- hashing (f2)
def test_sha256_oracle_fips180_vectors(golden_dir):
    import hashlib
    rows = _golden(golden_dir, "sha256_fips180.txt")
    msgs = {"EMPTY": b"", "MILLION_A": b"a" * 1000000}
    for spec, digest in rows:
        m = msgs.get(spec, spec.encode())
        assert hashlib.sha256(m).hexdigest() == digest
        # through the chunk interface: one chunk = the whole message
        if m:
            assert oracle.chunk_digests(np.frombuffer(m, np.uint8), [])[0].tobytes().hex() == digest


def test_chunk_digests_boundaries():
    data = synthgen.random_bytes(3, 1000)
    d = oracle.chunk_digests(data, [10, 500, 999])
    assert d.shape == (4, 32)
    import hashlib
    assert d[1].tobytes() == hashlib.sha256(data[10:500].tobytes()).digest()
    assert d[3].tobytes() == hashlib.sha256(data[999:].tobytes()).digest()



def test_size_bound_from_composes_over_pieces():
    """Running the rule piece by piece, each from the previous exit state, equals one run over the
    whole list (the streaming/sharded reading); the whole-stream case equals orc_size_bound."""
    rng = np.random.default_rng(8)
    for trial in range(200):
        n = int(rng.integers(2, 3000))
        cands = np.unique(rng.integers(1, n, int(rng.integers(0, 200)))).astype(np.uint64)
        mn = int(rng.integers(0, 60)); mx = int(rng.choice([0, max(1, mn) + int(rng.integers(0, 120))]))
        whole = oracle.size_bound(cands, n, mn, mx)
        w2, _, _ = oracle.size_bound_from(cands, n, True, 0, False, mn, mx)
        assert np.array_equal(whole, w2)
        bounds = sorted(set([0, n] + [int(x) for x in rng.integers(1, n, int(rng.integers(1, 5)))]))
        s, held, got = 0, False, []
        for a, b in zip(bounds[:-1], bounds[1:]):
            part = cands[(cands > a) & (cands <= b)]
            cuts, s, held = oracle.size_bound_from(part, b, b == n, s, held, mn, mx)
            got += cuts.tolist()
        assert got == whole.tolist(), (trial, mn, mx, bounds)


# --------------------------------------------------------------------------- sliced oracle runner
@pytest.mark.parametrize("n,sl,p", [
    ((3 << 20) + 77, 1 << 20, Params()),
    ((1 << 20) + 5, 65536, Params(divisor=256, magic=7)),
    (200000, 4096, Params(divisor=4, magic=3, window=5, poly=0x104C11DB7)),
    (4096 * 3, 4096, Params(divisor=2, magic=1)),
])
def test_candidates_stream_equals_whole(n, sl, p):
    """oracle.candidates_stream (slices with a w-1 overlap, used for the 16/64 GiB configs) ==
    oracle.candidates on the whole stream, including candidates at exactly a slice boundary."""
    whole = oracle.candidates(synthgen.random_bytes(11, n), p)
    parts, prev_b = [], 0
    for a, b, c in oracle.candidates_stream(11, n, p, slice_bytes=sl):
        assert a == prev_b and (c.size == 0 or (c[0] > a and c[-1] <= b))
        parts.append(c)
        prev_b = b
    assert prev_b == n
    got = np.concatenate(parts)
    assert np.array_equal(got, whole)
    # the dense-density parameter sets do hit slice boundaries exactly
    if p.divisor <= 4:
        assert any(int(c) % sl == 0 for c in whole)


def test_synthgen_fast_filler_matches_numpy_form():
    for off in (0, 3, 8, 12345, (1 << 36) + 5):
        for n in (0, 1, 7, 100, (3 << 20) | 5):
            assert np.array_equal(synthgen.random_bytes(9, n, off), synthgen.random_bytes_fast(9, n, off))


# --------------------------------------------------------------------------- matching index (f3)
def test_index_hand_built_duplicates():
    """oracle.Index against hand-worked set semantics (a chunk is new iff
    its hash was not seen before): digests A B A C B A with lengths 1..6 -> flags 1 1 0 1 0 0,
    3 new chunks of 1 + 2 + 4 bytes; a second batch C D -> 0 1."""
    A, B, C, D = (np.full(32, v, np.uint8) for v in (1, 2, 3, 4))
    ix = oracle.Index()
    f = ix.insert(np.stack([A, B, A, C, B, A]), [1, 2, 3, 4, 5, 6])
    assert f.tolist() == [1, 1, 0, 1, 0, 0]
    assert (ix.chunks, ix.new_chunks, ix.new_bytes) == (6, 3, 7)
    f = ix.insert(np.stack([C, D]), [10, 20])
    assert f.tolist() == [0, 1]
    assert (ix.chunks, ix.new_chunks, ix.new_bytes) == (8, 4, 27)
    # digests differing only in the last byte are distinct keys
    A2 = A.copy(); A2[31] ^= 1
    assert ix.insert(np.stack([A2]), [5]).tolist() == [1]


def test_index_snapshot_construction_closed_form():
    """Backup-style snapshots built at the digest level (the paper's similarity-table scheme,
    L1299-L1307): snapshot 0 = M distinct digests; snapshot s replaces each entry independently
    with probability p_s by a fresh digest.  By construction the distinct digests number
    M + sum_s R_s (R_s = entries replaced in snapshot s), so new_chunks and new_bytes are known
    without the index; also equal to numpy's unique row count."""
    rng = np.random.default_rng(5)
    M = 4000
    master = rng.integers(0, 256, (M, 32), dtype=np.uint8)
    lengths = rng.integers(1, 20000, M)
    ix = oracle.Index()
    ix.insert(master, lengths)
    exp_new, exp_bytes, allrows = M, int(lengths.sum()), [master]
    for s, p in enumerate([0.05, 0.10, 0.15, 0.20, 0.25, 0.05, 0.10, 0.15, 0.20], start=1):
        snap = master.copy()
        rep = rng.random(M) < p
        snap[rep] = rng.integers(0, 256, (int(rep.sum()), 32), dtype=np.uint8)
        flags = ix.insert(snap, lengths)
        assert np.array_equal(flags.astype(bool), rep)
        exp_new += int(rep.sum()); exp_bytes += int(lengths[rep].sum())
        allrows.append(snap)
    assert (ix.new_chunks, ix.new_bytes, ix.chunks) == (exp_new, exp_bytes, 10 * M)
    assert np.unique(np.concatenate(allrows), axis=0).shape[0] == exp_new
    # dedup ratio = logical / unique: 10 M / (M + sum R_s) ~ 10 / (1 + sum p) = 4.44
    assert abs(10 * M / exp_new - 10 / (1 + 1.25)) < 0.15

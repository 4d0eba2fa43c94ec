"""CPU oracle for Shredder's content-defined chunking (§2.1, §3.1).

TEST INFRASTRUCTURE ONLY. Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` leg / ``--impl reference`` arm may import this package. The product package
``paper_conf_fast_bhatotiarv12_b200`` never imports it and shares no code with it.

The arithmetic lives in ``oracle/rabin_oracle.c`` (plain C, compiled with gcc into
``oracle/liboracle.so``); this module only marshals arguments. ``oracle/brute.py`` holds the
pure-Python big-integer brute force that pins R1 on tiny inputs.

Functions (each cites the passage it follows; readings Q1..Q17 are listed in DESIGN.md):

* :func:`polymod` — R1, M(x) mod P(x) by long division (Eq. (1)).
* :func:`window_fp` / :func:`window_fps` — fingerprint of every full window (L444-L454, Q3/Q4/Q10).
* :func:`candidates` — {c = i+1 : fp_i mod D == r, c < N} (L447-L451, Q5-Q11); marker = 1
  gives the "mod p ... lower or equal to a constant" marker set of L249-L251.
* :func:`size_bound` — min/max rule (L259-L269, Q12-Q15).
* :func:`chunk` — candidates then size rule: the final cut offsets.
* :func:`is_irreducible` — Rabin's irreducibility test for ``div(x)`` (L255-L256).
* :func:`chunk_digests` — SHA-256 of every chunk (dedup step 2, L229-L238; §8(f) f2).

Parity status: every function is pinned (tests/test_oracle.py); parity with the *paper's own*
implementation is unpinned because the paper prints no fingerprint, polynomial or boundary.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from dataclasses import dataclass

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "rabin_oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")

LBFS_POLY = 0xBFE6B8A5BF378D83  # reading Q1: the LBFS polynomial, degree 63


def build(force: bool = False) -> str:
    """Compile oracle/rabin_oracle.c with gcc (plain C, -O2, pthreads)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + f".tmp{os.getpid()}"
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-fPIC", "-shared", "-pthread",
                               "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


_lib = None


def _L():
    global _lib
    if _lib is None:
        build()
        lib = ctypes.CDLL(_LIB)
        u64, u32, i64, cint = ctypes.c_uint64, ctypes.c_uint32, ctypes.c_int64, ctypes.c_int
        P = ctypes.c_void_p
        lib.orc_r1_mod.restype = u64
        lib.orc_r1_mod.argtypes = [P, u64, u64, cint]
        lib.orc_degree.restype = cint
        lib.orc_degree.argtypes = [u64]
        lib.orc_r1_window.restype = u64
        lib.orc_r1_window.argtypes = [P, u64, u32, u64]
        lib.orc_is_irreducible.restype = cint
        lib.orc_is_irreducible.argtypes = [u64]
        lib.orc_r2_tables.restype = P
        lib.orc_r2_tables.argtypes = [u32, u64]
        lib.orc_free.restype = None
        lib.orc_free.argtypes = [P]
        lib.orc_window_fps.restype = cint
        lib.orc_window_fps.argtypes = [P, u64, u32, u64, cint, P]
        lib.orc_candidates.restype = i64
        lib.orc_candidates.argtypes = [P, u64, u32, u64, u64, u64, cint, cint, cint, P, u64]
        lib.orc_size_bound.restype = i64
        lib.orc_size_bound.argtypes = [P, u64, u64, u64, u64, P, u64]
        lib.orc_size_bound_from.restype = i64
        lib.orc_size_bound_from.argtypes = [P, u64, u64, cint, u64, cint, u64, u64, P, u64, P]
        _lib = lib
    return _lib


@dataclass(frozen=True)
class Params:
    """Chunking parameters. Defaults are the paper's readings (Q1, Q5, Q6, Q15):
    P = LBFS polynomial (deg 63), w = 48 bytes (L444-L446), D = 2^13 ("low-order 13 bits",
    L447), r = 0x78, bounds off (min = 0, max = inf, L268-L269). ``max_size = 0`` = inf."""
    poly: int = LBFS_POLY
    window: int = 48
    divisor: int = 8192
    magic: int = 0x78
    min_size: int = 0
    max_size: int = 0
    marker: int = 0     # 0: fp mod D == r (L447-L451); 1: fp mod D <= r (L249-L251, variant f4)


def _bytes(data) -> np.ndarray:
    a = np.ascontiguousarray(np.frombuffer(data, dtype=np.uint8) if isinstance(data, (bytes, bytearray))
                             else np.asarray(data, dtype=np.uint8))
    return a


def degree(poly: int) -> int:
    return int(_L().orc_degree(poly))


def polymod(msg, poly: int, deg: int | None = None) -> int:
    """R1: M(x) mod P(x); msg[0] is the highest-degree byte, bit t of a byte = x^t (Q4).

    ``poly`` holds P with bit t = coeff of x^t. For a degree-64 P (CRC-64 pins) pass
    ``deg=64`` and ``poly`` = P - x^64."""
    a = _bytes(msg)
    if deg is None:
        deg = degree(poly)
        plow = poly ^ (1 << deg)
    else:
        plow = poly & ((1 << 64) - 1) if deg == 64 else poly ^ (1 << deg)
    return int(_L().orc_r1_mod(a.ctypes.data, a.size, plow, deg))


def window_fp(data, i: int, p: Params = Params()) -> int:
    """R1 fingerprint of the window ending at position i (Eq. (1), readings Q3/Q4)."""
    a = _bytes(data)
    assert p.window - 1 <= i < a.size
    return int(_L().orc_r1_window(a.ctypes.data, i, p.window, p.poly))


def window_fps(data, p: Params = Params(), method: int = 2) -> np.ndarray:
    """fp_i for every i in [w-1, N): index k holds fp_{k+w-1}. method 1 = R1, 2 = R2."""
    a = _bytes(data)
    n = max(0, a.size - p.window + 1)
    out = np.zeros(n, dtype=np.uint64)
    if n:
        rc = _L().orc_window_fps(a.ctypes.data, a.size, p.window, p.poly, method, out.ctypes.data)
        assert rc == 0
    return out


def r2_tables(p: Params = Params()) -> np.ndarray:
    """Positional tables C[j, b] = b(x) x^{8j} mod P, built with R1 (shape (w, 256))."""
    ptr = _L().orc_r2_tables(p.window, p.poly)
    assert ptr
    try:
        arr = np.ctypeslib.as_array(ctypes.cast(ptr, ctypes.POINTER(ctypes.c_uint64)),
                                    shape=(p.window * 256,)).copy()
    finally:
        _L().orc_free(ptr)
    return arr.reshape(p.window, 256)


def candidates(data, p: Params = Params(), method: int = 2, threads: int | None = None) -> np.ndarray:
    """Ascending cut candidates c = i+1 with fp_i mod D == r, w-1 <= i, c < N (L447-L451)."""
    a = _bytes(data)
    if threads is None:
        threads = len(os.sched_getaffinity(0))
    # output buffer sized from the expected count (hits per D positions: 1, or r + 1 for '<='), so
    # random-like inputs run the C routine once; a larger true count re-runs with the exact size
    # (round 1 started at 2^16 and ran every GiB-scale input twice, halving the measured rate)
    hits = (p.magic + 1) if p.marker else 1
    cap = max(1 << 16, int(2 * a.size * hits / p.divisor) + 4096)
    while True:
        out = np.zeros(cap, dtype=np.uint64)
        n = _L().orc_candidates(a.ctypes.data, a.size, p.window, p.poly, p.divisor, p.magic,
                                p.marker, method, threads, out.ctypes.data, cap)
        assert n >= 0, "oracle allocation failure"
        if n <= cap:
            return out[:n].copy()
        cap = int(n)


def candidates_stream(seed: int, n: int, p: Params = Params(), slice_bytes: int = 1 << 30,
                      threads: int | None = None):
    """Candidates of the first n bytes of the synthetic stream ``seed`` (synthgen), computed
    slice by slice so that GiB-scale configs fit in host memory (R2 over
    host slices with a w-1 byte overlap, the partition-with-overlap of PAPER.md L282-L287).

    Yields (a, b, cands) for consecutive slices: cands = every candidate c with a < c <= b
    (a = 0 for the first slice, whose lower end is the stream start), ascending, absolute.
    Slice [a, b) is evaluated on the stream bytes [a - (w-1), b + 1): its full windows end at
    i in [a, b - 1] (c = i + 1 in [a + 1, b]; c = b + 1 is excluded by c < N of the slice, and
    it is the next slice's first candidate position).  The last slice ends at N = n, where
    c < n (reading Q11).  Pinned against :func:`candidates` on whole streams in
    tests/test_oracle.py::test_candidates_stream_equals_whole."""
    import synthgen
    import threading
    k = p.window - 1
    bounds = list(range(0, n, slice_bytes)) + [n]

    def load(j):
        a, b = bounds[j], bounds[j + 1]
        lo, hi = max(0, a - k), min(n, b + 1)
        return synthgen.random_bytes_fast(seed, hi - lo, lo), lo

    nxt = [None]

    def prefetch(j):
        nxt[0] = load(j)

    t = None
    cur = load(0) if len(bounds) > 1 else None
    for j in range(len(bounds) - 1):
        if j + 2 < len(bounds):
            t = threading.Thread(target=prefetch, args=(j + 1,))
            t.start()
        data, lo = cur
        a, b = bounds[j], bounds[j + 1]
        c = candidates(data, p, 2, threads) + np.uint64(lo)
        yield a, b, c[(c > np.uint64(a)) & (c <= np.uint64(b))]
        if t is not None:
            t.join()
            t = None
            cur = nxt[0]


def bucket_digests(cuts: np.ndarray, n: int, bucket: int = 1 << 30) -> list[list]:
    """[count, sha256 hex] of the ascending offsets c with j*bucket < c <= (j+1)*bucket, for
    every bucket j covering [1, n): a compact exact record of a GiB-scale cut list (the
    little-endian u64 bytes of each bucket are hashed), so full-size results can be compared
    element by element against oracle values stored by tools/oracle_fullsize.py."""
    import hashlib
    c = np.ascontiguousarray(cuts, dtype="<u8")
    nb = max(1, (n - 1 + bucket - 1) // bucket)
    idx = np.searchsorted(c, np.arange(0, nb + 1, dtype=np.uint64) * np.uint64(bucket), side="right")
    out = []
    for j in range(nb):
        part = c[idx[j]:idx[j + 1]]
        out.append([int(part.size), hashlib.sha256(part.tobytes()).hexdigest()])
    return out


def size_bound(cands: np.ndarray, n: int, min_size: int, max_size: int) -> np.ndarray:
    """The min/max rule over ascending candidates (L259-L269, Q12-Q15); max_size 0 = inf."""
    c = np.ascontiguousarray(cands, dtype=np.uint64)
    cap = c.size + (n // max_size + 1 if max_size else 0) + 1
    out = np.zeros(cap, dtype=np.uint64)
    k = _L().orc_size_bound(c.ctypes.data, c.size, n, min_size, max_size, out.ctypes.data, cap)
    assert 0 <= k <= cap
    return out[:k].copy()


def size_bound_from(cands: np.ndarray, end: int, fin: bool, s0: int, held0: bool, min_size: int,
                    max_size: int) -> tuple[np.ndarray, int, bool]:
    """The size rule from an entry state over one stream range ending at `end` (a fed piece or
    a byte-range shard): returns (cuts, exit s, exit held).  size_bound(c, N, ..) ==
    size_bound_from(c, N, True, 0, False, ..)[0]."""
    c = np.ascontiguousarray(cands, dtype=np.uint64)
    cap = c.size + (end // max_size + 2 if max_size else 0) + 2
    out = np.zeros(cap, dtype=np.uint64)
    st = np.zeros(2, dtype=np.uint64)
    k = _L().orc_size_bound_from(c.ctypes.data, c.size, end, int(fin), s0, int(held0), min_size, max_size,
                                 out.ctypes.data, cap, st.ctypes.data)
    assert 0 <= k <= cap
    return out[:k].copy(), int(st[0]), bool(st[1])


def chunk(data, p: Params = Params(), method: int = 2, threads: int | None = None) -> np.ndarray:
    """Final cut offsets: candidates, then the size rule if min > 0 or max < inf."""
    a = _bytes(data)
    c = candidates(a, p, method, threads)
    if p.min_size == 0 and p.max_size == 0:
        return c
    return size_bound(c, a.size, p.min_size, p.max_size)


def chunk_digests(data, cuts) -> np.ndarray:
    """SHA-256 of every chunk [0,c0), [c0,c1), ..., [c_{n-1}, N) (dedup step 2, PAPER.md
    L229-L238).  The library routine hashlib.sha256 is the step (pinned by the
    FIPS 180 vectors in tests/golden/sha256_fips180.txt).  Returns (n+1, 32) uint8."""
    import hashlib
    a = _bytes(data)
    if a.size == 0:
        return np.zeros((0, 32), dtype=np.uint8)
    bounds = [0] + [int(c) for c in cuts] + [a.size]
    out = np.zeros((len(bounds) - 1, 32), dtype=np.uint8)
    mv = memoryview(a)
    for k in range(len(bounds) - 1):
        out[k] = np.frombuffer(hashlib.sha256(mv[bounds[k]:bounds[k + 1]]).digest(), dtype=np.uint8)
    return out


class Index:
    """Matching (dedup step 3, L235-L238): a set of digests; a chunk is new iff its digest was
    not seen before (plain Python set; test infrastructure)."""

    def __init__(self):
        self.seen = set()
        self.chunks = self.new_chunks = self.new_bytes = 0

    def insert(self, digests: np.ndarray, lengths) -> np.ndarray:
        flags = np.zeros(len(lengths), dtype=np.uint8)
        for k, (d, ln) in enumerate(zip(digests, lengths)):
            key = bytes(d)
            self.chunks += 1
            if key not in self.seen:
                self.seen.add(key)
                flags[k] = 1
                self.new_chunks += 1
                self.new_bytes += int(ln)
        return flags


def is_irreducible(poly: int) -> bool:
    """Rabin's irreducibility test for div(x) (L255-L256), degree 1..63."""
    return bool(_L().orc_is_irreducible(poly))

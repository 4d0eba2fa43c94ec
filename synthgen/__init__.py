"""Seeded synthetic inputs shared by the tests, the bench and the oracle checks.

This module holds NO chunking arithmetic (no fingerprint, table, marker or size rule): it only
produces bytes, so both sides (the CUDA product and the CPU oracle) can be fed identical input.
The device-side fill kernel in the product implements the same counter-based generator
independently; tests check the two agree byte for byte.

Counter-mode SplitMix64: 64-bit word k >= 0 of stream ``seed`` is
    x = seed + (k+1)*0x9E3779B97F4A7C15
    z = (x ^ x>>30) * 0xBF58476D1CE4E5B9 ; z = (z ^ z>>27) * 0x94D049BB133111EB ; z ^= z>>31
(all mod 2^64), stored little-endian at bytes 8k..8k+7. Any byte depends only on (seed, offset),
so a shard or a feed generates its own range (and its halo) without the rest of the stream.

Workload shapes (BASELINE.json configs; PAPER.md where the shape comes from):
* :func:`random_bytes`  — random data (configs 1, 3, 4).
* :func:`edited`        — a file plus a version with sparse inserts/deletes/overwrites (config 2;
  "small changes to the input lead to small changes in the set of chunks", L1150-L1153).
* :func:`snapshot`      — backup-style snapshots: 1 MiB segments of a master replaced with
  probability p (config 5; the paper's similarity-table scheme, p in 5-25 %
  from Fig. 18's x-axis L1342-L1351).
* :func:`text_like`     — words from a fixed 1,000-word list (skewed outgoing bytes).
* :func:`periodic`      — a repeated byte pattern, e.g. ``04 D5`` (adversarial candidate density).
"""
from __future__ import annotations

import numpy as np

GOLDEN = np.uint64(0x9E3779B97F4A7C15)
M1 = np.uint64(0xBF58476D1CE4E5B9)
M2 = np.uint64(0x94D049BB133111EB)
_BLOCK_WORDS = 1 << 22


def splitmix_words(seed: int, k0: int, count: int) -> np.ndarray:
    """Words k0 .. k0+count-1 of counter-mode SplitMix64 stream ``seed``."""
    out = np.empty(count, dtype=np.uint64)
    s = np.uint64(seed & 0xFFFFFFFFFFFFFFFF)
    with np.errstate(over="ignore"):
        for b in range(0, count, _BLOCK_WORDS):
            n = min(_BLOCK_WORDS, count - b)
            k = np.arange(k0 + b + 1, k0 + b + 1 + n, dtype=np.uint64)
            z = s + k * GOLDEN
            z = (z ^ (z >> np.uint64(30))) * M1
            z = (z ^ (z >> np.uint64(27))) * M2
            out[b:b + n] = z ^ (z >> np.uint64(31))
    return out


def random_bytes(seed: int, length: int, offset: int = 0) -> np.ndarray:
    """Bytes [offset, offset+length) of the SplitMix64 stream ``seed`` (uint8 array)."""
    if length <= 0:
        return np.zeros(0, dtype=np.uint8)
    k0 = offset // 8
    k1 = (offset + length + 7) // 8
    w = splitmix_words(seed, k0, k1 - k0)
    b = w.astype("<u8").view(np.uint8)
    s = offset - 8 * k0
    return b[s:s + length].copy()


def fill_random_into(buf: np.ndarray, seed: int, offset: int = 0, block: int = 1 << 26) -> None:
    """Write the stream ``seed`` starting at byte ``offset`` into ``buf`` (uint8, any size)."""
    n = buf.size
    for b in range(0, n, block):
        m = min(block, n - b)
        buf[b:b + m] = random_bytes(seed, m, offset + b)


_FILL_SRC = __import__("os").path.join(__import__("os").path.dirname(__file__), "splitmix_fill.c")
_FILL_LIB = _FILL_SRC[:-len("splitmix_fill.c")] + "libsplitmix.so"
_fill_lib = None


def _fill():
    """The multithreaded C filler (splitmix_fill.c, gcc), same stream definition as above."""
    global _fill_lib
    if _fill_lib is None:
        import ctypes
        import os
        import subprocess
        if not os.path.exists(_FILL_LIB) or os.path.getmtime(_FILL_LIB) < os.path.getmtime(_FILL_SRC):
            tmp = _FILL_LIB + f".tmp{os.getpid()}"
            subprocess.check_call(["gcc", "-O2", "-std=c11", "-fPIC", "-shared", "-pthread", "-o", tmp, _FILL_SRC])
            os.replace(tmp, _FILL_LIB)
        lib = ctypes.CDLL(_FILL_LIB)
        lib.sg_fill.restype = ctypes.c_int
        lib.sg_fill.argtypes = [ctypes.c_void_p, ctypes.c_uint64, ctypes.c_uint64, ctypes.c_uint64, ctypes.c_int]
        _fill_lib = lib
    return _fill_lib


def fill_fast(buf: np.ndarray, seed: int, offset: int = 0, threads: int | None = None) -> np.ndarray:
    """Bytes [offset, offset + buf.size) of stream ``seed`` into the contiguous uint8 ``buf``,
    multithreaded C (GB/s; the numpy form above is ~0.2 GB/s).  Returns ``buf``."""
    import os
    assert buf.dtype == np.uint8 and buf.flags["C_CONTIGUOUS"]
    if threads is None:
        threads = len(os.sched_getaffinity(0))
    if buf.size:
        _fill().sg_fill(buf.ctypes.data, buf.size, seed & 0xFFFFFFFFFFFFFFFF, offset, threads)
    return buf


def random_bytes_fast(seed: int, length: int, offset: int = 0) -> np.ndarray:
    """:func:`random_bytes` through the C filler."""
    return fill_fast(np.empty(max(0, length), dtype=np.uint8), seed, offset)


def _uniform(seed: int, count: int) -> np.ndarray:
    """``count`` doubles in [0,1) from the SplitMix64 stream ``seed`` (top 53 bits)."""
    w = splitmix_words(seed, 0, count)
    return (w >> np.uint64(11)).astype(np.float64) * (1.0 / (1 << 53))


def edited(base: np.ndarray, seed: int, n_edits: int = 100, min_gap: int = 64 * 1024,
           max_len: int = 4096) -> tuple[np.ndarray, list[tuple[int, str, int]]]:
    """A version of ``base`` with ``n_edits`` sparse edits (config 2 recipe).

    Positions: sorted, uniform over the file, at least ``min_gap`` apart. Operation: insert
    40 % / delete 40 % / overwrite 20 %; length U[1, max_len]; new bytes from SplitMix64(seed).
    Returns (new bytes, [(position in base, op, length)])."""
    n = base.size
    u = _uniform(seed ^ 0x5EED, 4 * n_edits + 16)
    usable = n - (n_edits + 1) * min_gap
    if usable <= 0:
        raise ValueError("input too small for the requested edits")
    raw = np.sort((u[:n_edits] * usable).astype(np.int64))
    pos = raw + np.arange(1, n_edits + 1, dtype=np.int64) * min_gap
    ops = []
    pieces = []
    prev = 0
    fresh_off = 0
    for e in range(n_edits):
        p = int(pos[e])
        ru = u[n_edits + e]
        op = "insert" if ru < 0.4 else ("delete" if ru < 0.8 else "overwrite")
        ln = 1 + int(u[2 * n_edits + e] * max_len)
        ln = min(ln, max_len)
        pieces.append(base[prev:p])
        if op == "insert":
            pieces.append(random_bytes(seed, ln, fresh_off)); fresh_off += ln
            prev = p
        elif op == "delete":
            prev = p + ln
        else:
            pieces.append(random_bytes(seed, ln, fresh_off)); fresh_off += ln
            prev = p + ln
        ops.append((p, op, ln))
    pieces.append(base[prev:])
    return np.concatenate(pieces), ops


SNAPSHOT_P = (0.0, 0.05, 0.10, 0.15, 0.20, 0.25, 0.05, 0.10, 0.15, 0.20)


def snapshot(master_seed: int, length: int, s: int, segment: int = 1 << 20) -> np.ndarray:
    """Backup snapshot ``s`` (0..9) of the master stream (config 5 recipe).

    Snapshot 0 is the master. For s >= 1 each ``segment``-byte segment is replaced
    independently with probability SNAPSHOT_P[s] by SplitMix64(100+s) bytes at the same offset."""
    out = random_bytes(master_seed, length)
    if s == 0:
        return out
    nseg = (length + segment - 1) // segment
    u = _uniform(1000 + s, nseg)
    for g in np.nonzero(u < SNAPSHOT_P[s])[0]:
        a = int(g) * segment
        b = min(length, a + segment)
        out[a:b] = random_bytes(100 + s, b - a, a)
    return out


def text_like(seed: int, length: int, n_words: int = 1000) -> np.ndarray:
    """Words (2-10 lowercase letters) from a fixed 1,000-word list, space separated."""
    rnd = splitmix_words(seed ^ 0x7E47, 0, n_words * 11)
    words = []
    for k in range(n_words):
        L = 2 + int(rnd[k * 11] % np.uint64(9))
        words.append(bytes(97 + int(rnd[k * 11 + 1 + j] % np.uint64(26)) for j in range(L)) + b" ")
    lens = np.array([len(x) for x in words])
    avg = float(lens.mean())
    picks = splitmix_words(seed, 0, int(length / avg * 1.2) + 64) % np.uint64(n_words)
    buf = b"".join(words[int(i)] for i in picks)
    while len(buf) < length:
        buf += buf
    return np.frombuffer(buf[:length], dtype=np.uint8).copy()


def periodic(pattern: bytes, length: int) -> np.ndarray:
    """``pattern`` repeated to ``length`` bytes (e.g. b'\\x04\\xd5': a candidate every 2 bytes)."""
    reps = length // len(pattern) + 1
    return np.frombuffer(pattern * reps, dtype=np.uint8)[:length].copy()

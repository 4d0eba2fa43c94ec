"""Host planning logic (no GPU): the slot map that splits a job's window ends into the edge CTA's
head/tail segments and the hot kernel's rows (csrc/shred.cu plan_map, through the C-ABI test hook
shred_debug_plan).

Invariants checked over random lengths, stream offsets, source alignments and SM counts:
* the head segments, the rows and the tail segments tile [t_begin, t_end) exactly, in order
  (every window end is tested once: parity with the oracle depends on it);
* the bulk region starts 16-byte aligned in memory (TMA) and at least 16*ceil(w/16) bytes into
  the job's bytes (the rows' warm-up reads them), or at the stream start itself when the job
  starts there with no carry (virtual zero bytes before it);
* rows are a multiple of 32 bytes (whole 32-byte TMA rounds; a loop iteration of two rounds may
  stop after the first);
* the edge CTA has one thread per head and per tail segment;
* slot groups fit the scatter kernel's table, and per-slot lists hold >= 2x the expected count.
"""
import ctypes

import numpy as np
import pytest

K63, K32, GENERIC = 1, 2, 3
MAX_GROUPS = 4096
GEN_THREADS = 256


@pytest.fixture(scope="module")
def L():
    from paper_conf_fast_bhatotiarv12_b200 import _build
    lib = ctypes.CDLL(_build.build())
    f = lib.shred_debug_plan
    u64 = ctypes.c_uint64
    f.argtypes = [ctypes.c_int, ctypes.c_int, ctypes.c_int, u64, u64, u64, u64, u64, ctypes.c_uint32, ctypes.c_int,
                  ctypes.POINTER(u64)]
    f.restype = ctypes.c_int
    return lib


def plan(L, path, small_ok, sms, addr, p_begin, t_begin, t_end, divisor=8192, window=48, zero_lead=0):
    out = (ctypes.c_uint64 * 16)()
    rc = L.shred_debug_plan(path, small_ok, sms, addr, p_begin, t_begin, t_end, divisor, window, zero_lead, out)
    assert rc == 0
    keys = ("bulk", "small", "head_start", "head_seg", "n_head", "b0", "S", "nrows", "tail_start",
            "tail_seg", "n_tail", "nc", "ngroups", "rows_cta", "cap", "edge_threads")
    return dict(zip(keys, list(out)))


def segments(m, t_begin, t_end):
    """The window-end ranges of every slot, in slot order (kernels.cuh slot_range)."""
    out = []
    lim = m["b0"] if m["nrows"] else (m["tail_start"] if m["n_tail"] else t_end)
    for i in range(m["n_head"]):
        a = m["head_start"] + i * m["head_seg"]
        out.append((a, min(a + m["head_seg"], lim)))
    for r in range(m["nrows"]):
        a = m["b0"] + r * m["S"]
        out.append((a, a + m["S"]))
    for i in range(m["n_tail"]):
        a = m["tail_start"] + i * m["tail_seg"]
        out.append((a, min(a + m["tail_seg"], t_end)))
    return out


def check(m, path, addr, p_begin, t_begin, t_end, divisor=8192, window=48, zero_lead=0):
    segs = segments(m, t_begin, t_end)
    pos = t_begin
    for a, b in segs:
        assert a == pos and b >= a, (a, b, pos)
        pos = b
    assert pos == t_end
    assert all(b > a for a, b in segs) or t_end == t_begin
    if m["bulk"]:
        assert path in (K63, K32)
        assert (addr + (m["b0"] - p_begin)) % 16 == 0
        # each row warms up on the 16*ceil(w/16) bytes before it, inside the job's bytes, or it
        # starts at the stream start itself (no carry: virtual zero bytes before it)
        warm = 16 * ((window + 15) // 16)
        assert m["b0"] >= t_begin
        assert m["b0"] >= p_begin + warm or (zero_lead and m["b0"] == p_begin == t_begin)
        assert m["S"] % 32 == 0 and m["S"] >= 32 and m["nrows"] >= 1
        assert m["n_head"] <= m["edge_threads"] and m["n_tail"] <= m["edge_threads"]
        assert m["nc"] == -(-m["nrows"] // m["rows_cta"])
        assert m["ngroups"] == m["nc"] + 2
        longest = max(m["S"], m["tail_seg"])
    else:
        assert m["nrows"] == 0 and m["n_tail"] == 0
        assert m["ngroups"] == -(-m["n_head"] // GEN_THREADS)
        longest = m["head_seg"]
    assert m["ngroups"] <= MAX_GROUPS
    assert m["cap"] == min(4096, 2 * longest // divisor + 16)


@pytest.mark.parametrize("path", [K63, K32, GENERIC])
def test_plan_tiles_every_window_end_once(L, path):
    rng = np.random.default_rng(path)
    lengths = [0, 1, 47, 48, 255, 4095, 4096, 4097, 70001, 1 << 20, (1 << 20) + 4093, 5 << 20,
               (1 << 30) + 12345, 1 << 36]
    for n in lengths + [int(x) for x in rng.integers(1, 1 << 28, 40)]:
        for _ in range(3):
            addr = int(rng.integers(0, 1 << 20)) * 16 + int(rng.integers(0, 16))
            p_begin = int(rng.integers(0, 1 << 40))
            t_begin = p_begin + int(rng.integers(0, 200))
            sms = int(rng.choice([1, 2, 132, 148, 160]))
            small_ok = int(rng.integers(0, 2))
            window = int(rng.choice([1, 16, 17, 47, 48, 64, 65, 100, 4096]))
            zl = int(rng.integers(0, 2)) if window <= 64 else 0      # long windows: never a zero lead
            if window > 64:
                small_ok = 0                                          # no small shape for them
            if zl and rng.integers(0, 2):
                t_begin = p_begin
            m = plan(L, path, small_ok, sms, addr, p_begin, t_begin, t_begin + n, window=window, zero_lead=zl)
            check(m, path, addr, p_begin, t_begin, t_begin + n, window=window, zero_lead=zl)


def test_plan_shapes(L):
    """1 GiB on 148 SMs: one wave of 147 bulk CTAs x 1024 rows + the edge CTA; 1 MiB takes the
    small launch shape; below 4 KiB (or on the generic path) there are no rows."""
    m = plan(L, K63, 1, 148, 0, 0, 47, 1 << 30)
    assert m["bulk"] and not m["small"] and m["nc"] == 147 and m["rows_cta"] == 1024
    assert m["S"] % 32 == 0 and m["nrows"] * m["S"] <= (1 << 30)
    m = plan(L, K63, 1, 148, 0, 0, 47, 1 << 20)
    assert m["bulk"] and m["small"] and m["rows_cta"] == 256
    m = plan(L, K63, 0, 148, 0, 0, 47, 1 << 20)
    assert m["bulk"] and not m["small"]
    assert not plan(L, K63, 1, 148, 0, 0, 0, 4000)["bulk"]
    assert not plan(L, GENERIC, 1, 148, 0, 0, 0, 1 << 30)["bulk"]
    # an aligned stream from its start, no carry: the rows begin at byte 0, no head segments;
    # 1 MiB = 32768 rows of 32 B, no tail either (the edge CTA has nothing to roll)
    m = plan(L, K63, 1, 148, 0, 0, 0, 1 << 20, zero_lead=1)
    assert m["b0"] == 0 and m["n_head"] == 0 and m["n_tail"] == 0 and m["S"] == 32
    m = plan(L, K63, 1, 148, 0, 0, 0, 1 << 20, zero_lead=0)
    assert m["b0"] == 48 and m["n_head"] == 3


def test_plan_rejects_inconsistent_arguments(L):
    out = (ctypes.c_uint64 * 16)()
    assert L.shred_debug_plan(K63, 1, 148, 0, 100, 50, 1000, 8192, 48, 0, out) != 0   # t_begin < p_begin
    assert L.shred_debug_plan(K63, 1, 148, 0, 0, 10, 5, 8192, 48, 0, out) != 0        # t_end < t_begin
    assert L.shred_debug_plan(K63, 1, 0, 0, 0, 0, 5, 8192, 48, 0, out) != 0           # no SMs
    assert L.shred_debug_plan(K63, 1, 148, 0, 0, 0, 5, 8192, 4097, 0, out) != 0       # w > 4096
    assert L.shred_debug_plan(K63, 1, 148, 0, 0, 0, 5, 8192, 4096, 0, out) == 0       # long window

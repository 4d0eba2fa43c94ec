"""Parameter validation and kernel-path selection of the C-ABI library (no GPU): shred_check_params
runs shred_init's validation and path choice without a device.

* The library's irreducibility test (Ben-Or, csrc/shred.cu) must agree with the oracle's
  independent Rabin test (pinned by Gauss's counts in test_oracle.py) on random polynomials of
  every degree 8..63: a reducible P would make "fingerprint" ill-defined as a field element.
* The documented parameter ranges (include/shred.h) are enforced.
* The path table: which parameters run on the u64 / u32 hot kernel, with which marker kind.
"""
import ctypes

import numpy as np
import pytest

import oracle

K63, K32, GENERIC = 1, 2, 3
MK_EQ, MK_LE, MK_DIV, MK_REM = 0, 1, 2, 3
LBFS = 0xBFE6B8A5BF378D83


@pytest.fixture(scope="module")
def check():
    from paper_conf_fast_bhatotiarv12_b200 import _binding, _build
    lib = ctypes.CDLL(_build.build())
    f = lib.shred_check_params
    f.argtypes = [ctypes.POINTER(_binding._Params), ctypes.POINTER(ctypes.c_int), ctypes.POINTER(ctypes.c_int)]
    f.restype = ctypes.c_int

    def run(**kw):
        p = _binding.Params(**kw)._c()
        path, mk = ctypes.c_int(-9), ctypes.c_int(-9)
        rc = f(ctypes.byref(p), ctypes.byref(path), ctypes.byref(mk))
        return rc, path.value, mk.value
    return run


def test_irreducibility_agrees_with_the_oracle(check):
    rng = np.random.default_rng(11)
    seen = {True: 0, False: 0}
    for deg in range(8, 64):
        for _ in range(12):
            low = int(rng.integers(0, 1 << min(deg, 62))) | 1
            if deg > 62:
                low |= int(rng.integers(0, 2)) << 62
            P = (1 << deg) | (low & ((1 << deg) - 1))
            irr = oracle.is_irreducible(P)
            rc, _, _ = check(poly=P, divisor=2, magic=0)
            assert (rc == 0) == irr, hex(P)
            seen[irr] += 1
    assert seen[True] > 20 and seen[False] > 20
    for P in (LBFS, 0x104C11DB7, (1 << 63) | 3, 0x11D):        # known irreducible
        assert check(poly=P, divisor=2, magic=0)[0] == 0
    for P in ((1 << 63) | 1, (1 << 63) | (1 << 5) | (1 << 2) | 1):   # an even number of terms: (x+1) divides
        assert check(poly=P, divisor=2, magic=0)[0] != 0


def test_parameter_ranges(check):
    assert check()[0] == 0
    bad = [dict(poly=0xFF), dict(window=0), dict(window=4097), dict(marker=2), dict(divisor=1, magic=0),
           dict(poly=0x104C11DB7, divisor=1 << 33), dict(divisor=(1 << 63) + 2, magic=0),
           dict(divisor=8192, magic=8192), dict(min_size=100, max_size=99), dict(min_size=0, max_size=0)]
    for kw in bad[:-1]:
        assert check(**kw)[0] != 0, kw
    assert check(**bad[-1])[0] == 0                          # bounds off
    assert check(window=4096)[0] == 0 and check(poly=0x104C11DB7, divisor=1 << 32, magic=5)[0] == 0
    assert check(divisor=1 << 63, magic=0)[0] == 0           # D = 2^deg


@pytest.mark.parametrize("kw,path,mk", [
    (dict(), K63, MK_EQ),                                                # the paper's reading
    (dict(marker=1, magic=3), K63, MK_LE),
    (dict(window=47), K63, MK_EQ), (dict(window=64), K63, MK_EQ), (dict(window=1), K63, MK_EQ),
    (dict(window=65), K63, MK_EQ), (dict(window=4096), K63, MK_EQ), (dict(window=47, marker=1, magic=1), K63, MK_LE),
    (dict(divisor=10000, magic=7), K63, MK_DIV), (dict(divisor=3 << 31, magic=7), K63, MK_DIV),
    (dict(divisor=1 << 32, magic=7), K63, MK_EQ), (dict(divisor=1 << 33, magic=7), K63, MK_REM),
    (dict(divisor=3 << 32, magic=7), K63, MK_REM), (dict(divisor=10000, magic=7, marker=1), K63, MK_REM),
    (dict(divisor=1 << 40, magic=7, marker=1), K63, MK_REM), (dict(window=65, divisor=10000, magic=7, marker=1), K63, MK_REM),
    (dict(poly=0x104C11DB7, divisor=1000, magic=999, marker=1), K32, MK_REM),
    (dict(poly=0x104C11DB7), K32, MK_EQ), (dict(poly=0x104C11DB7, divisor=10000, magic=3), K32, MK_DIV),
    (dict(poly=0x11D, divisor=64, magic=1), K32, MK_EQ),                         # degree 8: byte index
    (dict(poly=(1 << 40) | 0x39, divisor=1024, magic=5), K63, MK_EQ),            # degree 40: u64 state
])
def test_path_table(check, kw, path, mk):
    if "poly" in kw and not oracle.is_irreducible(kw["poly"]):
        pytest.skip("not irreducible")
    rc, p, m = check(**kw)
    assert rc == 0 and (p, m) == (path, mk), (kw, p, m)


def test_k32t_multiplier_equals_the_reduction_table():
    """K32T (T[t] as one integer product): for every eligible P (deg <= 32, Q = P - x^k with terms
    >= 8 apart below k - 7) the library's multiplier gives, for every byte t,
    t * M mod 2^32 == (t(x) x^k mod P) XOR (t << k mod 2^32): the reduction computed here by the
    oracle's long division (R1), the cancel term by the definition of the u32 shift.  Ineligible
    polynomials (overlapping copies of t, or a term too high) are refused."""
    from paper_conf_fast_bhatotiarv12_b200 import _build
    lib = ctypes.CDLL(_build.build())
    f = lib.shred_debug_tprod
    f.argtypes = [ctypes.c_uint64, ctypes.POINTER(ctypes.c_uint32), ctypes.POINTER(ctypes.c_uint32)]
    f.restype = ctypes.c_int
    eligible = [0x80002001, 0x80040001, 0x40200001, 0x40000201, 0x10000201, 0x10002001, 0x800201,
                0x804001, 0x40201]
    for P in eligible:
        assert oracle.is_irreducible(P)
        m = ctypes.c_uint32(0)
        assert f(P, ctypes.byref(m), None) == 1, hex(P)
        k = P.bit_length() - 1
        for t in range(256):
            # t(x) x^k mod P by R1 on the message t || zero bits: shift t by k bits via bytes
            msg = t << k
            nb = (msg.bit_length() + 7) // 8 or 1
            red = oracle.polymod(np.frombuffer(msg.to_bytes(nb, "big"), np.uint8), P)
            exp = red ^ ((t << k) & 0xFFFFFFFF)
            assert (t * m.value) & 0xFFFFFFFF == exp, (hex(P), t)
    for P in (0x104C11DB7, LBFS, 0x8000000B, 0x80000081, 0x20000005, (1 << 31) | (1 << 24) | 1):
        assert f(P, None, None) == 0, hex(P)
    # K63T (deg 41..63): T[t] = (t * mult_hi mod 2^32) : (t * mult) == t(x) x^k mod P ^ (t << k mod 2^64)
    for P in (0x8000000000000801,):
        assert oracle.is_irreducible(P)
        m, mh = ctypes.c_uint32(0), ctypes.c_uint32(0)
        assert f(P, ctypes.byref(m), ctypes.byref(mh)) == 1
        k = P.bit_length() - 1
        for t in range(256):
            msg = t << k
            red = oracle.polymod(np.frombuffer(msg.to_bytes((msg.bit_length() + 7) // 8 or 1, "big"), np.uint8), P)
            exp = red ^ ((t << k) & 0xFFFFFFFFFFFFFFFF)
            got = (((t * mh.value) & 0xFFFFFFFF) << 32) | ((t * m.value) & 0xFFFFFFFF)
            assert got == exp, t
    # deg 41..63 with a term too high for the low word, or too close: refused
    for P in (LBFS, (1 << 63) | (1 << 25) | 1, (1 << 63) | (1 << 7) | 1, (1 << 50) | (1 << 30) | 1):
        assert f(P, None, None) == 0, hex(P)

"""Pure-Python big-integer brute force — pins the C oracle's R1 on tiny inputs.

TEST INFRASTRUCTURE ONLY (see oracle/__init__.py). Independent of rabin_oracle.c: the
window is turned into ONE Python integer (int.from_bytes, big-endian: the oldest byte is the
most significant, bit t of the newest byte is x^t — reading Q4) and reduced by polynomial
long division over GF(2) on arbitrary-precision integers (Eq. (1)).
"""
from __future__ import annotations


def gf2_mod(a: int, p: int) -> int:
    """a(x) mod p(x) over GF(2), both as Python ints (bit t = coeff of x^t)."""
    dp = p.bit_length() - 1
    while a and a.bit_length() - 1 >= dp:
        a ^= p << (a.bit_length() - 1 - dp)
    return a


def window_fp(window: bytes, p: int) -> int:
    return gf2_mod(int.from_bytes(bytes(window), "big"), p)


def candidates(data: bytes, p: int, w: int, D: int, r: int, marker: int = 0) -> list[int]:
    """Every c = i+1 with w-1 <= i, c < N and fp_i mod D == r (readings Q9-Q11); marker = 1:
    fp_i mod D <= r (the "lower or equal to a constant" marker set, L249-L251)."""
    data = bytes(data)
    out = []
    for i in range(w - 1, len(data) - 1):
        v = window_fp(data[i + 1 - w:i + 1], p) % D
        if (v <= r) if marker else (v == r):
            out.append(i + 1)
    return out

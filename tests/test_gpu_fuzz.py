"""Seeded randomized parity sweep: the CUDA path (through the C ABI) vs the CPU oracle on random
parameter sets, inputs, lengths, alignments and API paths, element by element.

Each case draws (from one fixed seed, so the ids are stable and a failure reproduces by id):
* P: the paper's LBFS polynomial (K63), the sparse trinomials the multiply-reduction kernels take
  (K32T x^31+x^13+1, K63T x^63+x^11+1), 0x104C11DB7 (K32B), x^31+x^3+1 (K32, T table),
  x^8+x^4+x^3+x^2+1 (degree 8), or a dense random irreducible of degree 9..63 (L255-L258: "an
  irreducible polynomial div(x) of degree k", k left open);
* w in 1..64 (hot kernel, register pops) or 65..200 (hot kernel, pops from a second TMA tile);
* D = 2^m ('==' and '<=', L447-L451 / L249-L251) or any other D (remainder kernels, reading Q8);
* r < D; min/max bounds on or off (the size rule of §8(c));
* the input: SplitMix64 bytes, text-like words, a short periodic pattern, or zeros;
  length 0..3.5 MiB (windows > 64 below 400 KiB), base offset 0..15;
* the call: one-shot `shred_chunk`; `shred_feed` in random pieces (pinned host or device, ring of
  2-3 slots) + `shred_flush`; or G = 2..5 byte-range shards (`shred_candidates_range` with the
  min(w-1, start) halo) concatenated, then the global size rule (`shred_size_bound`).
The oracle is R2 (direct per-window reduction, positional tables built by long division)."""
import os

import numpy as np
import pytest
import torch

import oracle
import synthgen

pytestmark = pytest.mark.gpu

# fixed by default (stable ids); SHRED_FUZZ_N / SHRED_FUZZ_SEED run a wider sweep ad hoc
N_CASES = int(os.environ.get("SHRED_FUZZ_N", 512))
SEED = int(os.environ.get("SHRED_FUZZ_SEED", 20261018))
POOL = {
    "k63_lbfs": oracle.LBFS_POLY,
    "k32t": 0x80002001,
    "k63t": 0x8000000000000801,
    "k32b": 0x104C11DB7,
    "k32_table": 0x80000009,
    "deg8": 0x11D,
}


def _deg(p: int) -> int:
    return p.bit_length() - 1


def _dense_irreducible(rng) -> int:
    deg = int(rng.integers(9, 64))
    while True:
        low = int(rng.integers(0, 1 << min(deg, 62))) | 1
        p = (1 << deg) | (low & ((1 << deg) - 1))
        if oracle.is_irreducible(p):
            return p


def _cases():
    rng = np.random.default_rng(SEED)
    out = []
    for i in range(N_CASES):
        c = {}
        kind = list(POOL) + ["dense"]
        pk = kind[int(rng.integers(0, len(kind)))]
        c["poly"] = _dense_irreducible(rng) if pk == "dense" else POOL[pk]
        deg = _deg(c["poly"])
        if rng.random() < 0.8:
            c["window"] = int(rng.choice([1, 2, 3, 7, 8, 15, 16, 17, 31, 32, 33, 47, 48, 49, 63, 64]))
        else:
            c["window"] = int(rng.integers(65, 201))
        if rng.random() < 0.7:
            m = int(rng.integers(1, min(deg, 16) + 1))
            c["divisor"] = 1 << m
        else:
            while True:
                d = int(rng.integers(3, 40000))
                if d & (d - 1) and d <= (1 << deg):
                    break
            c["divisor"] = d
        c["marker"] = int(rng.random() < 0.25)
        D = c["divisor"]
        c["magic"] = int(rng.integers(0, max(1, D // 16) + 1)) if c["marker"] else int(rng.integers(0, D))
        c["min_size"], c["max_size"] = 0, 0
        if rng.random() < 0.35:
            mn = int(rng.integers(1, 3000)) if rng.random() < 0.7 else 0
            mx = int(rng.integers(max(mn, 1) + 1, 100000)) if rng.random() < 0.7 else 0
            if mn == 0 and mx == 0:
                mx = 8192
            c["min_size"], c["max_size"] = mn, mx
        u = rng.random()
        c["data"] = "random" if u < 0.6 else "text" if u < 0.75 else "periodic" if u < 0.9 else "zeros"
        u = rng.random()
        n = int(rng.integers(0, 5000)) if u < 0.3 else int(rng.integers(5000, 600000)) if u < 0.7 \
            else int(rng.integers(600000, 3584 * 1024))
        if c["window"] > 64:
            n = min(n, 400000)
        c["n"] = n
        c["offset"] = int(rng.integers(0, 16))
        u = rng.random()
        c["api"] = "chunk" if u < 0.5 else "feed" if u < 0.75 else "shards"
        c["seed"] = int(rng.integers(0, 1 << 30))
        out.append(c)
    return out


CASES = _cases()


def _id(c):
    b = f"{c['min_size']}-{c['max_size']}" if (c["min_size"] or c["max_size"]) else "nob"
    return (f"p{c['poly']:x}-w{c['window']}-D{c['divisor']}{'le' if c['marker'] else 'eq'}{c['magic']}-{b}-"
            f"{c['data']}{c['n']}+{c['offset']}-{c['api']}")


def _data(c) -> np.ndarray:
    n, s = c["n"], c["seed"]
    if c["data"] == "random":
        return synthgen.random_bytes(s, n)
    if c["data"] == "text":
        return synthgen.text_like(s, n)
    if c["data"] == "periodic":
        rng = np.random.default_rng(s)
        pat = bytes(rng.integers(0, 256, int(rng.integers(1, 9)), dtype=np.uint8))
        return synthgen.periodic(pat, n)
    return np.zeros(n, np.uint8)


def _dev(a: np.ndarray, offset: int) -> torch.Tensor:
    buf = torch.empty(a.size + offset + 64, dtype=torch.uint8, device="cuda")
    t = buf[offset:offset + a.size]
    t.copy_(torch.from_numpy(a))
    return t


@pytest.fixture(scope="module")
def pkg():
    import paper_conf_fast_bhatotiarv12_b200 as P
    return P


@pytest.mark.parametrize("c", CASES, ids=[_id(c) for c in CASES])
def test_random_case(pkg, c):
    data = _data(c)
    n = data.size
    p = pkg.Params(poly=c["poly"], window=c["window"], divisor=c["divisor"], magic=c["magic"],
                   min_size=c["min_size"], max_size=c["max_size"], marker=c["marker"])
    op = oracle.Params(p.poly, p.window, p.divisor, p.magic, p.min_size, p.max_size, p.marker)
    exp = oracle.chunk(data, op)
    ch = pkg.Chunker(p)
    rng = np.random.default_rng(c["seed"] ^ 0x5EED)
    if c["api"] == "chunk":
        got = ch.chunk(_dev(data, c["offset"])).cpu().numpy().astype(np.uint64)
    elif c["api"] == "feed":
        ch.set_ring(int(rng.integers(2, 4)), int(rng.choice([1 << 16, 1 << 18, 1 << 20])))
        outs, off, k = [], 0, 0
        while off < n:
            s = int(min(n - off, rng.choice([1, 2, c["window"] - 1 or 1, c["window"], 4093, 65536,
                                              (1 << 18) + 7, 1 << 20])))
            piece = torch.from_numpy(data[off:off + s].copy())
            x = piece.pin_memory() if k % 2 == 0 else piece.cuda()
            outs.append(ch.feed(x).cpu().numpy())
            off += s
            k += 1
        outs.append(ch.flush().cpu().numpy())
        got = np.concatenate(outs).astype(np.uint64)
    else:
        G = int(rng.integers(2, 6))
        cuts = sorted(int(v) for v in rng.integers(0, n + 1, G - 1)) if n else [0] * (G - 1)
        bounds = [0] + cuts + [n]
        parts = []
        for g in range(G):
            a, b = bounds[g], bounds[g + 1]
            if a == b:
                continue
            halo = min(c["window"] - 1, a)
            parts.append(ch.candidates_range(_dev(data[a - halo:b], c["offset"]), halo, a, n).cpu().numpy())
        cand = np.concatenate(parts).astype(np.uint64) if parts else np.zeros(0, np.uint64)
        assert np.array_equal(cand, oracle.candidates(data, op))
        if c["min_size"] or c["max_size"]:
            got = ch.size_bound(torch.from_numpy(cand.astype(np.int64)).cuda(), n).cpu().numpy().astype(np.uint64)
        else:
            got = cand
    assert got.size == exp.size, (got.size, exp.size)
    assert np.array_equal(got, exp)

"""Small cases of every kernel path, for compute-sanitizer (memcheck / racecheck / synccheck;
tools/sanitize.sh).  Test infrastructure (kept under tests/ because it calls the oracle): checks
results against the oracle too, so a silent corruption under the tool is caught."""
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import oracle  # noqa: E402
import synthgen  # noqa: E402
import paper_conf_fast_bhatotiarv12_b200 as pkg  # noqa: E402


def check(ch, data, off=0):
    buf = torch.zeros(data.size + off + 64, dtype=torch.uint8, device="cuda")
    x = buf[off:off + data.size]
    x.copy_(torch.from_numpy(data))
    got = ch.chunk(x).cpu().numpy().astype(np.uint64)
    p = ch.params
    exp = oracle.chunk(data, oracle.Params(p.poly, p.window, p.divisor, p.magic, p.min_size, p.max_size, p.marker))
    assert np.array_equal(got, exp), (p, data.size)


def main():
    n = (1 << 20) + 333
    data = synthgen.random_bytes(1, n)
    check(pkg.Chunker(pkg.Params()), data, 3)
    check(pkg.Chunker(pkg.Params(divisor=64, magic=5)), data)
    check(pkg.Chunker(pkg.Params(poly=0x104C11DB7)), data, 1)
    check(pkg.Chunker(pkg.Params(window=32)), data[:200000])
    check(pkg.Chunker(pkg.Params(min_size=2048, max_size=65536)), data)
    check(pkg.Chunker(pkg.Params()), synthgen.periodic(b"\x04\xd5", 300000))
    check(pkg.Chunker(pkg.Params(min_size=3)), synthgen.periodic(b"\x04\xd5", 100000))
    check(pkg.Chunker(pkg.Params(divisor=10000, magic=1234)), data, 5)          # MK_DIV
    check(pkg.Chunker(pkg.Params(window=47, divisor=4096, magic=9, marker=1)), data[:300000], 2)   # funnel, '<='
    check(pkg.Chunker(pkg.Params(window=65)), data[:100000])                       # long window
    check(pkg.Chunker(pkg.Params(window=200, marker=1, magic=3, divisor=1024)), data[:300000], 3)   # long window '<=', funnel
    check(pkg.Chunker(pkg.Params(divisor=12345, magic=3, marker=1)), data[:400000], 7)   # MK_REM, u64
    check(pkg.Chunker(pkg.Params(divisor=3 << 32, magic=77)), data[:300000], 1)          # MK_REM '=='
    check(pkg.Chunker(pkg.Params(poly=0x104C11DB7, divisor=1000, magic=2, marker=1)), data[:300000])  # MK_REM, u32
    check(pkg.Chunker(pkg.Params(poly=0x11D, window=20, divisor=256, magic=9)), data[:300000], 4)      # degree 8
    check(pkg.Chunker(pkg.Params(poly=0x80002001)), data)                                 # K32T, aligned start (no head)
    check(pkg.Chunker(pkg.Params(poly=0x80002001, window=31, marker=1, magic=3)), data[:300000], 9)    # K32T funnel '<='
    check(pkg.Chunker(pkg.Params()), data[: (1 << 20)])                                 # small shape, 32-B rows
    check(pkg.Chunker(pkg.Params(poly=0x80002001, magic=0)), data, 2)       # K32T, r = 0: zero-filled rows past nrows are markers
    check(pkg.Chunker(pkg.Params(poly=0x80002001, marker=1, magic=1)), data[:700001], 1)   # K32T '<=' (packed hit masks)
    check(pkg.Chunker(pkg.Params(divisor=4096, magic=77, marker=1)), data[:500000], 6)   # '<=' lists sized by rate
    # f2 / f3: SHA-256 of every chunk (hashlib oracle) and the dedup index
    chh = pkg.Chunker(pkg.Params())
    x = torch.from_numpy(data).cuda()
    cuts = chh.chunk(x)
    dig = chh.hash_chunks(x, cuts).cpu().numpy()
    assert np.array_equal(dig, oracle.chunk_digests(data, cuts.cpu().numpy().astype(np.uint64)))
    # batched hashing over two buffers, one of them at an unaligned address
    x2 = torch.from_numpy(data[1:200001].copy()).cuda()
    c2 = chh.chunk(x2)
    n1 = torch.tensor([cuts.numel()], dtype=torch.int64, device="cuda")
    n2 = torch.tensor([c2.numel()], dtype=torch.int64, device="cuda")
    d1 = torch.empty((cuts.numel() + 1) * 32, dtype=torch.uint8, device="cuda")
    d2 = torch.empty((c2.numel() + 1) * 32, dtype=torch.uint8, device="cuda")
    dig2 = chh.hash_chunks(x2, c2).cpu().numpy()                  # one unaligned buffer (ws kernel)
    chh.hash_chunks_batch_async([(x, cuts, n1, d1), (x2, c2, n2, d2)])
    torch.cuda.synchronize()
    assert np.array_equal(d1.view(-1, 32).cpu().numpy(), dig)
    assert np.array_equal(d2.view(-1, 32).cpu().numpy(),
                          oracle.chunk_digests(data[1:200001], c2.cpu().numpy().astype(np.uint64)))
    assert np.array_equal(d2.view(-1, 32).cpu().numpy(), dig2)
    chh.index_reset(1 << 12)
    n_c = torch.tensor([cuts.numel()], dtype=torch.int64, device="cuda")
    chh.index_insert_async(torch.from_numpy(dig.reshape(-1)).cuda(), cuts, n_c, data.size)
    torch.cuda.synchronize()
    assert chh.index_stats()["chunks"] == dig.shape[0]
    ch = pkg.Chunker(pkg.Params(divisor=1024, min_size=256, max_size=4096))
    ch.set_ring(2, 1 << 18)
    outs = []
    for a, b in ((0, 1000), (1000, 700001), (700001, n)):
        outs.append(ch.feed(torch.from_numpy(data[a:b].copy()).pin_memory()).cpu().numpy())
    outs.append(ch.flush().cpu().numpy())
    got = np.concatenate(outs).astype(np.uint64)
    assert np.array_equal(got, oracle.chunk(data, oracle.Params(divisor=1024, min_size=256, max_size=4096)))
    torch.cuda.synchronize()
    print("sanitize cases ok")


if __name__ == "__main__":
    main()

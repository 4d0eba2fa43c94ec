"""f2: SHA-256 of every chunk on the GPU vs the oracle (hashlib per chunk, FIPS-180-pinned)."""
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


def test_padding_edge_lengths(pkg):
    """Chunk lengths around the 55/56/64-byte padding edges, 1-byte chunks, unaligned starts."""
    lens = [1, 1, 2, 3, 54, 55, 56, 57, 63, 64, 65, 119, 120, 121, 127, 128, 129, 1000, 4095, 4096, 4097]
    rng = np.random.default_rng(3)
    lens = lens + [int(x) for x in rng.integers(1, 3000, 200)]
    cuts = np.cumsum(lens)[:-1]
    n = int(np.sum(lens))
    data = synthgen.random_bytes(5, n)
    ch = pkg.Chunker(pkg.Params())
    got = ch.hash_chunks(torch.from_numpy(data).cuda(), torch.from_numpy(cuts.astype(np.int64)).cuda())
    exp = oracle.chunk_digests(data, cuts)
    assert np.array_equal(got.cpu().numpy(), exp)


@pytest.mark.parametrize("shift", [1, 2, 3, 5])
def test_unaligned_input_pointer(pkg, shift):
    """d_in = a slice x[shift:] of a device buffer (base address not 4-byte aligned): the word
    loads align on the absolute address, and the chunk ending at the buffer end
    reads no word past its allocation."""
    lens = [1, 3, 55, 56, 64, 65, 127, 128, 129, 4096, 4097] + [int(v) for v in np.random.default_rng(shift).integers(1, 5000, 150)]
    cuts = np.cumsum(lens)[:-1]
    n = int(np.sum(lens))
    data = synthgen.random_bytes(6, n + shift)
    base = torch.from_numpy(data).cuda()
    x = base[shift:]
    assert x.data_ptr() % 4 != 0 or shift % 4 == 0
    ch = pkg.Chunker(pkg.Params())
    got = ch.hash_chunks(x, torch.from_numpy(cuts.astype(np.int64)).cuda())
    assert np.array_equal(got.cpu().numpy(), oracle.chunk_digests(data[shift:], cuts))
    # and the chunker itself on the same unaligned slice
    assert np.array_equal(ch.chunk(x).cpu().numpy().astype(np.uint64), oracle.candidates(data[shift:]))


def test_single_chunk_and_fips_message(pkg):
    ch = pkg.Chunker(pkg.Params())
    for m in (b"abc", b"abcdbcdecdefdefgefghfghighijhijkijkljklmklmnlmnomnopnopq", b"a" * 1000000):
        x = torch.frombuffer(bytearray(m), dtype=torch.uint8).cuda()
        got = ch.hash_chunks(x, torch.zeros(0, dtype=torch.int64).cuda())
        assert got.shape == (1, 32)
        assert np.array_equal(got.cpu().numpy(), oracle.chunk_digests(np.frombuffer(m, np.uint8), []))


def test_batched_buffers_one_work_list(pkg):
    """shred_hash_chunks_batch: 19 buffers (more than one launch of 16) of different lengths and
    chunkings, one repeated, each chunk's digest == hashlib (FIPS-180-pinned) of that buffer's
    chunk; chunk counts read on the device."""
    rng = np.random.default_rng(12)
    ch = pkg.Chunker(pkg.Params(divisor=1024))
    jobs, exp = [], []
    datas = [synthgen.random_bytes(40 + k, int(rng.integers(1, 300000))) for k in range(18)] + [None]
    datas[-1] = datas[3]
    for k, data in enumerate(datas):
        x = torch.from_numpy(data).cuda()
        if k % 3 == 0:                       # the chunker's own cuts (device count)
            cuts = torch.empty(max(1, data.size // 256), dtype=torch.int64, device="cuda")
            nc = torch.zeros(1, dtype=torch.int64, device="cuda")
            ch.chunk_async(x, cuts, nc)
            torch.cuda.synchronize()
            c = cuts[:int(nc.item())].cpu().numpy()
        else:                                # arbitrary cuts incl. 1-byte and padding-edge chunks
            c = np.unique(rng.integers(1, max(2, data.size), int(rng.integers(0, 60)))).astype(np.int64)
            cuts = torch.from_numpy(c).cuda() if c.size else torch.zeros(1, dtype=torch.int64, device="cuda")
            nc = torch.tensor([c.size], dtype=torch.int64, device="cuda")
        dig = torch.empty((c.size + 1) * 32, dtype=torch.uint8, device="cuda")
        jobs.append((x, cuts, nc, dig))
        exp.append(oracle.chunk_digests(data, c))
    ch.hash_chunks_batch_async(jobs)
    torch.cuda.synchronize()
    for (x, cuts, nc, dig), e in zip(jobs, exp):
        assert np.array_equal(dig.view(-1, 32).cpu().numpy(), e)


@pytest.mark.parametrize("bounded", [False, True])
def test_chunk_then_hash_on_device(pkg, bounded):
    """Chunking -> hashing chained on one stream (the cut count never leaves the device)."""
    n = (8 << 20) + 333
    data = synthgen.random_bytes(7, n)
    p = pkg.Params(divisor=2048, min_size=512 if bounded else 0, max_size=16384 if bounded else 0)
    ch = pkg.Chunker(p)
    x = torch.from_numpy(data).cuda()
    cuts = torch.empty(n // 256, dtype=torch.int64, device="cuda")
    ncut = torch.zeros(1, dtype=torch.int64, device="cuda")
    dig = torch.empty(n // 256 * 32, dtype=torch.uint8, device="cuda")
    ch.chunk_async(x, cuts, ncut)
    ch.hash_chunks_async(x, cuts, ncut, dig)
    torch.cuda.synchronize()
    k = int(ncut.item())
    c = cuts[:k].cpu().numpy()
    assert np.array_equal(c.astype(np.uint64), oracle.chunk(data, oracle.Params(divisor=2048, min_size=p.min_size,
                                                                                 max_size=p.max_size)))
    assert np.array_equal(dig[:(k + 1) * 32].view(-1, 32).cpu().numpy(), oracle.chunk_digests(data, c))


# ------------------------------------------------------------------ f3: dedup across snapshots
def test_index_dedup_across_snapshots_vs_oracle(pkg):
    """chunk -> hash -> index over backup snapshots (configs[4] recipe, 12 MiB master): new-chunk
    and new-byte counts equal the oracle's set semantics; per-chunk flags agree except among
    identical digests inserted by the same call (then exactly one is new)."""
    import tools.snapshots as S
    n = 12 << 20
    ch = pkg.Chunker(pkg.Params(divisor=4096))
    ch.index_reset(1 << 20)
    oi = oracle.Index()
    buf = torch.empty(n, dtype=torch.uint8, device="cuda")
    cuts = torch.empty(n // 512, dtype=torch.int64, device="cuda")
    ncut = torch.zeros(1, dtype=torch.int64, device="cuda")
    dig = torch.empty(n // 512 * 32, dtype=torch.uint8, device="cuda")
    flags = torch.empty(n // 512, dtype=torch.uint8, device="cuda")
    for s in (0, 1, 3, 5, 0, 9):                                  # snapshot 0 twice: all duplicates
        S.build_snapshot(buf, 6, s)
        ch.chunk_async(buf, cuts, ncut)
        ch.hash_chunks_async(buf, cuts, ncut, dig)
        ch.index_insert_async(dig, cuts, ncut, n, flags)
        torch.cuda.synchronize()
        k = int(ncut.item())
        c = cuts[:k].cpu().numpy()
        d = dig[:(k + 1) * 32].view(-1, 32).cpu().numpy()
        lens = np.diff(np.concatenate([[0], c, [n]]))
        exp_flags = oi.insert(d, lens)
        got_flags = flags[:k + 1].cpu().numpy()
        st = ch.index_stats()
        assert (st["chunks"], st["new_chunks"], st["new_bytes"], st["full"]) == \
               (oi.chunks, oi.new_chunks, oi.new_bytes, 0)
        uniq_batch = {bytes(x) for x in d}
        if len(uniq_batch) == len(d):                             # no duplicates inside the batch
            assert np.array_equal(got_flags, exp_flags)


@pytest.mark.parametrize("shift", [0, 1, 3])
@pytest.mark.parametrize("last", [1, 55, 56, 63, 64, 65, 119, 128])
def test_last_chunk_at_buffer_end(pkg, shift, last):
    """The padding blocks of the chunk that ends at the buffer's last byte: the word loads stop at
    the last word that starts inside the buffer, whatever the alignment (one buffer and batched)."""
    lens = [100, 64, 7, last]
    cuts = np.cumsum(lens)[:-1]
    n = int(np.sum(lens))
    data = synthgen.random_bytes(11 + last, n + shift)
    base = torch.from_numpy(data).cuda()
    x = base[shift:]
    ch = pkg.Chunker(pkg.Params())
    c = torch.from_numpy(cuts.astype(np.int64)).cuda()
    exp = oracle.chunk_digests(data[shift:], cuts)
    assert np.array_equal(ch.hash_chunks(x, c).cpu().numpy(), exp)
    nc = torch.tensor([c.numel()], dtype=torch.int64, device="cuda")
    d = [torch.empty((c.numel() + 1) * 32, dtype=torch.uint8, device="cuda") for _ in range(2)]
    ch.hash_chunks_batch_async([(x, c, nc, d[0]), (x, c, nc, d[1])])
    torch.cuda.synchronize()
    for di in d:
        assert np.array_equal(di.view(-1, 32).cpu().numpy(), exp)

"""Multi-GPU byte-range sharding.

Rank g of G owns the window ends [start_g, end_g) of one stream of `total_len` bytes and holds
its bytes plus the w-1 = 47 bytes before them (the halo: "a small overlap of the size of the
sliding window (w bytes) near partition boundaries", L282-L287).  Candidates are independent
per shard; the only exchange is:

* C2 - an all-gather of the per-rank candidate counts (8 B per rank) -> each rank's exclusive
  prefix = the index of its first candidate in the global list (unbounded mode, the paper's
  default: nothing else is exchanged);
* bounded mode (min/max set), the distributed size rule (default): every rank
  runs the rule over its own candidates from an entry state (s = last cut, held); ranks
  all-gather their exit states (16 B per rank) and re-run from their predecessor's exit until
  no entry changes (Jacobi on the chain of shard states: exact after at most G rounds since rank
  r's entry is exact after round r; usually 2 rounds because runs from different entries
  coincide within a few candidates);
* C3 - bounded mode, `mode="gather"`: an all-gather of the candidate lists (padded to the
  largest count), then the sequential size rule over the concatenation on every rank.

The collectives go through ``torch.distributed`` (NCCL on GPUs; gloo in the CPU tests, where
device tensors are staged through host memory).  The per-shard compute is an *engine*: the
product uses :class:`paper_conf_fast_bhatotiarv12_b200.Chunker` (CUDA, via the C ABI); the CPU
tests plug in an oracle-backed engine instead.

Host synchronisation.  With an engine that has the asynchronous calls (the Chunker:
``candidates_range_async``, ``size_bound_state_dev``), the unbounded path enqueues the shard's
chunking and the count all-gather and returns without synchronising the host: counts, the
rank's base index and the total stay device tensors until a caller reads ``base``/``total``/
``local``.  The chain mode runs its first two rounds back to back on the device and
synchronises once to learn whether a third is needed (a host round trip per
round before).  Engines without the asynchronous calls take the synchronous path.
"""
from __future__ import annotations

import torch
import torch.distributed as dist


def shard_bounds(total_len: int, world: int, rank: int, align: int = 4096) -> tuple[int, int]:
    """[start, end) of rank's window ends: contiguous ranges, starts rounded down to `align`."""
    def cut(g):
        if g <= 0:
            return 0
        if g >= world:
            return total_len
        return (total_len * g // world) // align * align
    return cut(rank), cut(rank + 1)


def halo_of(start: int, window: int = 48) -> int:
    return min(window - 1, start)


def _gloo(group) -> bool:
    return dist.get_backend(group) == "gloo"


def _all_gather(out: torch.Tensor, inp: torch.Tensor, group=None) -> None:
    """all_gather_into_tensor; gloo gets host copies of device tensors."""
    if inp.is_cuda and _gloo(group):
        o = torch.empty(out.shape, dtype=out.dtype)
        dist.all_gather_into_tensor(o, inp.cpu(), group=group)
        out.copy_(o)
    else:
        dist.all_gather_into_tensor(out, inp, group=group)


def _all_reduce_max(t: torch.Tensor, group=None) -> None:
    if t.is_cuda and _gloo(group):
        h = t.cpu()
        dist.all_reduce(h, op=dist.ReduceOp.MAX, group=group)
        t.copy_(h)
    else:
        dist.all_reduce(t, op=dist.ReduceOp.MAX, group=group)


def exchange_halo(own: torch.Tensor, start: int, window: int = 48, group=None) -> torch.Tensor:
    """C1 for real (non-regenerable) data: rank g gets the last min(w-1, start) bytes of the
    bytes before its shard from its predecessor, and returns [halo || own] ready for
    chunk_sharded.  The exchange is one all-gather of each rank's (w-1)-byte tail
    ((w-1) x world bytes over NCCL/NVLink; ranks must hold contiguous shards in rank order and a
    shard shorter than w-1 bytes must not follow another short one)."""
    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    k = window - 1
    tail = torch.zeros(k, dtype=torch.uint8, device=own.device)
    m = min(k, own.numel())
    if m:
        tail[k - m:] = own[own.numel() - m:]
    allt = torch.zeros(world * k, dtype=torch.uint8, device=own.device)
    _all_gather(allt, tail, group)
    halo = min(k, start)
    if rank == 0 or halo == 0:
        return own.contiguous()
    prev = allt.view(world, k)[rank - 1]
    return torch.cat([prev[k - halo:], own]).contiguous()


class ShardResult:
    """One rank's share of a sharded chunking.  Device tensors; the int views synchronise.

    local    this rank's candidates (absolute offsets, ascending)
    base     index of local[0] in the global candidate list     (base_t: device 0-d int64)
    total    global number of candidates                        (total_t)
    counts   per-rank candidate counts (int64, on the collective's device)
    cuts     bounded: this rank's cuts ("chain") or all cuts ("gather")
    cut_base bounded "chain": index of cuts[0] in the global cut list (cut_base_t)
    rounds   bounded "chain": state-exchange rounds run
    """

    def __init__(self, local_buf, n_local, counts, rank):
        self._local_buf, self._n_local = local_buf, n_local
        self.counts = counts
        self.base_t = counts[:rank].sum()
        self.total_t = counts.sum()
        self._cut_buf = self._n_cut = None
        self.cut_base_t = None
        self.cuts_all = None
        self.rounds = 0
        self._redo = None            # exact synchronous re-run if the candidate buffer overflowed

    @property
    def local(self) -> torch.Tensor:
        n = int(self._n_local.reshape(-1)[0])
        if n > self._local_buf.numel():
            if self._redo is None:
                raise RuntimeError(f"candidate buffer overflow: {n} > {self._local_buf.numel()}")
            self._local_buf = self._redo()
            self._n_local = torch.tensor([self._local_buf.numel()], dtype=torch.int64)
            self._redo = None
            return self._local_buf
        return self._local_buf[:n]

    @property
    def base(self) -> int:
        return int(self.base_t)

    @property
    def total(self) -> int:
        return int(self.total_t)

    @property
    def cuts(self):
        if self.cuts_all is not None:
            return self.cuts_all
        if self._cut_buf is None:
            return None
        return self._cut_buf[:int(self._n_cut.reshape(-1)[0])]

    @property
    def cut_base(self) -> int:
        return 0 if self.cut_base_t is None else int(self.cut_base_t)


def _expected_cap(engine, n: int) -> int:
    """A candidate-buffer capacity for n window ends that random-like data does not exceed
    (2x the expectation + slack); overflow is detected and redone exactly."""
    p = engine.params
    rate = (p.magic + 1 if getattr(p, "marker", 0) else 1) / p.divisor
    return int(min(max(1, n), 2 * n * rate + 4096))


def chunk_sharded(x: torch.Tensor, halo: int, start: int, total_len: int, engine,
                  group=None, bounded: bool | None = None, mode: str = "chain",
                  cap: int | None = None) -> ShardResult:
    """Chunk this rank's shard `x` (= stream bytes [start - halo, start + len(x) - halo)).

    engine: ``params`` (min_size, max_size, ...) and either the asynchronous calls
    ``candidates_range_async(x, halo, start, total_len, out, n_out)`` and
    ``size_bound_state_dev(cands, n_cand, end, fin, state_in, out, n_out, state_out)``, or the
    synchronous ``candidates_range(x, halo, start, total_len) -> int64 tensor`` and
    ``size_bound_state(cands, end, fin, s, held) -> (cuts, s, held)``; ``size_bound(cands,
    total_len)`` for mode "gather".  Bounded mode: "chain" (the distributed size rule, this
    rank's cuts) or "gather" (C3, every rank gets all cuts)."""
    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    p = engine.params
    if bounded is None:
        bounded = bool(p.min_size or p.max_size)
    ln = x.numel() - halo
    end = start + ln
    fin = end == total_len
    asyn = hasattr(engine, "candidates_range_async")
    if asyn:
        dev = x.device
        cap = _expected_cap(engine, ln) if cap is None else cap
        local_buf = torch.empty(max(1, cap), dtype=torch.int64, device=dev)
        n_local = torch.zeros(1, dtype=torch.int64, device=dev)
        engine.candidates_range_async(x, halo, start, total_len, local_buf, n_local)
    else:
        local_buf = engine.candidates_range(x, halo, start, total_len)
        dev = local_buf.device
        n_local = torch.tensor([local_buf.numel()], dtype=torch.int64, device=dev)
    counts = torch.zeros(world, dtype=torch.int64, device=dev)
    _all_gather(counts, n_local, group)                         # C2
    res = ShardResult(local_buf, n_local, counts, rank)
    if asyn:
        res._redo = lambda: engine.candidates_range(x, halo, start, total_len)
    if not bounded:
        return res
    if mode == "gather":
        cs = counts.cpu().tolist()
        local = res.local
        mx = max(cs) if cs else 0
        pad = torch.zeros(max(1, mx), dtype=torch.int64, device=dev)
        pad[:local.numel()] = local
        allp = torch.zeros(world * max(1, mx), dtype=torch.int64, device=dev)
        _all_gather(allp, pad, group)
        allp = allp.view(world, max(1, mx))
        cat = torch.cat([allp[g, :cs[g]] for g in range(world)]) if sum(cs) else allp.new_zeros(0)
        res.cuts_all = engine.size_bound(cat.contiguous(), total_len)
        return res
    if not asyn:
        return _chain_sync(res, engine, start, end, fin, group, world, rank, dev)
    # ---- chain, on the device: entry guess "the predecessor's last candidate was accepted"
    nl = n_local.clamp(max=local_buf.numel())
    last = torch.where(nl > 0, local_buf[(nl - 1).clamp(min=0)], torch.full_like(nl, -1))
    lasts = torch.zeros(world, dtype=torch.int64, device=dev)
    _all_gather(lasts, last, group)
    entry = torch.zeros(2, dtype=torch.int64, device=dev)
    if rank > 0:
        prev = lasts[:rank]
        idx = torch.where(prev >= 0, torch.arange(rank, device=dev), torch.full_like(prev, -1)).max()
        s0 = torch.where(idx >= 0, prev[idx.clamp(min=0)], torch.zeros_like(idx))
        entry[0] = s0
        entry[1] = ((idx >= 0) & (s0 == start)).to(torch.int64)
    mx = p.max_size
    span = ln + (mx if mx else 0)
    ccap = local_buf.numel() + (span // mx + 3 if mx else 2)
    if p.min_size:
        ccap = min(ccap, span // p.min_size + 2)
    cut_buf = torch.empty(max(1, ccap), dtype=torch.int64, device=dev)
    n_cut = torch.zeros(1, dtype=torch.int64, device=dev)
    exit_ = torch.zeros(2, dtype=torch.int64, device=dev)
    exits = torch.zeros(2 * world, dtype=torch.int64, device=dev)
    flag = torch.zeros(1, dtype=torch.int64, device=dev)
    rnd = 0
    while True:
        rnd += 1
        engine.size_bound_state_dev(local_buf, n_local, end, fin, entry, cut_buf, n_cut, exit_)
        _all_gather(exits, exit_, group)
        new_entry = exits.view(world, 2)[rank - 1] if rank > 0 else torch.zeros(2, dtype=torch.int64, device=dev)
        # "changed" of any rank, plus overflow of a candidate or cut buffer (-> exact redo)
        flag[0] = (new_entry != entry).any().to(torch.int64) | (n_local[0] > local_buf.numel()).to(torch.int64) * 2 \
            | (n_cut[0] > cut_buf.numel()).to(torch.int64) * 2
        entry.copy_(new_entry)
        if rnd < 2 and rnd < world:
            continue                                          # round 2 runs without a host check
        _all_reduce_max(flag, group)
        f = int(flag.item())
        if f & 2:
            return chunk_sharded(x, halo, start, total_len, engine, group, bounded, mode,
                                 cap=max(cap * 4, ln + 1) if f & 2 else cap)
        if f == 0 or rnd >= world:
            break
    ncs = torch.zeros(world, dtype=torch.int64, device=dev)
    _all_gather(ncs, n_cut, group)
    res._cut_buf, res._n_cut = cut_buf, n_cut
    res.cut_base_t = ncs[:rank].sum()
    res.rounds = rnd
    return res


def _chain_sync(res, engine, start, end, fin, group, world, rank, dev):
    """The chain mode with a synchronous engine (host-side entry states)."""
    local = res.local
    last = torch.tensor([int(local[-1]) if local.numel() else -1], dtype=torch.int64, device=dev)
    lasts = torch.zeros(world, dtype=torch.int64, device=dev)
    _all_gather(lasts, last, group)
    lv = lasts.cpu().tolist()
    prev = [v for v in lv[:rank] if v >= 0]
    entry = (0, False) if rank == 0 or not prev else (prev[-1], prev[-1] == start)
    for rnd in range(1, world + 1):
        cuts, s_out, h_out = engine.size_bound_state(local, end, fin, entry[0], entry[1])
        ex = torch.tensor([s_out, int(h_out)], dtype=torch.int64, device=dev)
        exits = torch.zeros(2 * world, dtype=torch.int64, device=dev)
        _all_gather(exits, ex, group)
        ev = exits.view(world, 2).cpu().tolist()
        new_entry = (0, False) if rank == 0 else (ev[rank - 1][0], bool(ev[rank - 1][1]))
        changed = torch.tensor([int(new_entry != entry)], dtype=torch.int64, device=dev)
        _all_reduce_max(changed, group)                      # any rank's entry changed?
        if int(changed.item()) == 0:
            break
        entry = new_entry
    nc = torch.tensor([cuts.numel()], dtype=torch.int64, device=dev)
    ncs = torch.zeros(world, dtype=torch.int64, device=dev)
    _all_gather(ncs, nc, group)
    res.cuts_all = cuts
    res.cut_base_t = ncs[:rank].sum()
    res.rounds = rnd
    return res


def gather_all(res: ShardResult, group=None) -> torch.Tensor:
    """Concatenate every rank's local candidates (rank order) on every rank."""
    world = dist.get_world_size(group)
    cs = res.counts.cpu().tolist()
    local = res.local
    mx = max(1, max(cs) if cs else 0)
    pad = torch.zeros(mx, dtype=torch.int64, device=local.device)
    pad[:local.numel()] = local
    allp = torch.zeros(world * mx, dtype=torch.int64, device=local.device)
    _all_gather(allp, pad, group)
    allp = allp.view(world, mx)
    return torch.cat([allp[g, :cs[g]] for g in range(world)])

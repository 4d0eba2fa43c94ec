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

The collectives go through ``torch.distributed`` (NCCL on GPUs; gloo in the CPU tests).  The
per-shard compute is an *engine*: the product uses :class:`paper_conf_fast_bhatotiarv12_b200.Chunker`
(CUDA, via the C ABI); the CPU tests plug in an oracle-backed engine instead.
"""
from __future__ import annotations

from dataclasses import dataclass

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
    dist.all_gather_into_tensor(allt, tail, group=group)
    halo = min(k, start)
    if rank == 0 or halo == 0:
        return own.contiguous()
    prev = allt.view(world, k)[rank - 1]
    return torch.cat([prev[k - halo:], own]).contiguous()


@dataclass
class ShardResult:
    local: torch.Tensor          # this rank's candidates (absolute offsets, ascending)
    base: int                    # index of local[0] in the global candidate list
    total: int                   # global number of candidates
    counts: torch.Tensor         # per-rank counts (int64, on the collective's device)
    cuts: torch.Tensor | None = None   # bounded: this rank's cuts ("chain") or all cuts ("gather")
    cut_base: int = 0            # bounded "chain": index of cuts[0] in the global cut list
    rounds: int = 0              # bounded "chain": state-exchange rounds until convergence


def chunk_sharded(x: torch.Tensor, halo: int, start: int, total_len: int, engine,
                  group=None, bounded: bool | None = None, mode: str = "chain") -> ShardResult:
    """Chunk this rank's shard `x` (= stream bytes [start - halo, start + len(x) - halo)).

    engine: has ``candidates_range(x, halo, start, total_len) -> int64 tensor``,
    ``size_bound(cands, total_len) -> int64 tensor``, ``size_bound_state(cands, end, fin, s,
    held) -> (cuts, s, held)`` and ``params`` (min_size, max_size).  Bounded mode: "chain" (the
    distributed size rule, this rank's cuts) or "gather" (C3, every rank gets all cuts)."""
    world = dist.get_world_size(group)
    rank = dist.get_rank(group)
    if bounded is None:
        bounded = bool(engine.params.min_size or engine.params.max_size)
    local = engine.candidates_range(x, halo, start, total_len)
    dev = local.device
    n = torch.tensor([local.numel()], dtype=torch.int64, device=dev)
    counts = torch.zeros(world, dtype=torch.int64, device=dev)
    dist.all_gather_into_tensor(counts, n, group=group)            # C2
    cs = counts.cpu().tolist()
    base = int(sum(cs[:rank]))
    total = int(sum(cs))
    res = ShardResult(local=local, base=base, total=total, counts=counts)
    if not bounded:
        return res
    if mode == "chain":
        end = start + x.numel() - halo
        fin = end == total_len
        # entry guess: "the predecessor's last candidate was accepted" (its last candidates are
        # all-gathered, 8 B per rank); rank 0 starts from the exact stream-start state
        last = torch.tensor([int(local[-1]) if local.numel() else -1], dtype=torch.int64, device=dev)
        lasts = torch.zeros(world, dtype=torch.int64, device=dev)
        dist.all_gather_into_tensor(lasts, last, group=group)
        lv = lasts.cpu().tolist()
        prev = [v for v in lv[:rank] if v >= 0]
        entry = (0, False) if rank == 0 or not prev else (prev[-1], prev[-1] == start)
        for rnd in range(1, world + 1):
            cuts, s_out, h_out = engine.size_bound_state(local, end, fin, entry[0], entry[1])
            ex = torch.tensor([s_out, int(h_out)], dtype=torch.int64, device=dev)
            exits = torch.zeros(2 * world, dtype=torch.int64, device=dev)
            dist.all_gather_into_tensor(exits, ex, group=group)
            ev = exits.view(world, 2).cpu().tolist()
            new_entry = (0, False) if rank == 0 else (ev[rank - 1][0], bool(ev[rank - 1][1]))
            changed = torch.tensor([int(new_entry != entry)], dtype=torch.int64, device=dev)
            dist.all_reduce(changed, group=group)                 # any rank's entry changed?
            if int(changed.item()) == 0:
                break
            entry = new_entry
        nc = torch.tensor([cuts.numel()], dtype=torch.int64, device=dev)
        ncs = torch.zeros(world, dtype=torch.int64, device=dev)
        dist.all_gather_into_tensor(ncs, nc, group=group)
        res.cuts = cuts
        res.cut_base = int(sum(ncs.cpu().tolist()[:rank]))
        res.rounds = rnd
        return res
    # C3: all-gather the (padded) candidate lists, then the global size rule (replicated)
    mx = max(cs) if cs else 0
    pad = torch.zeros(max(1, mx), dtype=torch.int64, device=dev)
    pad[:local.numel()] = local
    allp = torch.zeros(world * max(1, mx), dtype=torch.int64, device=dev)
    dist.all_gather_into_tensor(allp, pad, group=group)
    allp = allp.view(world, max(1, mx))
    cat = torch.cat([allp[g, :cs[g]] for g in range(world)]) if total else allp.new_zeros(0)
    res.cuts = engine.size_bound(cat.contiguous(), total_len)
    return res


def gather_all(res: ShardResult, group=None) -> torch.Tensor:
    """Concatenate every rank's local candidates (rank order) on every rank."""
    world = dist.get_world_size(group)
    cs = res.counts.cpu().tolist()
    mx = max(1, max(cs) if cs else 0)
    pad = torch.zeros(mx, dtype=torch.int64, device=res.local.device)
    pad[:res.local.numel()] = res.local
    allp = torch.zeros(world * mx, dtype=torch.int64, device=res.local.device)
    dist.all_gather_into_tensor(allp, pad, group=group)
    allp = allp.view(world, mx)
    return torch.cat([allp[g, :cs[g]] for g in range(world)])

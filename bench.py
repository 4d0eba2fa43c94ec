#!/usr/bin/env python
"""Benchmark: content-defined chunking throughput on B200 (BASELINE.json metric).

python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]

Workload (configs[1] of BASELINE.json, per GPU): a 1 GiB synthetic file (bytes
[rank GiB, (rank+1) GiB) of the SplitMix64 stream seed 2, so ranks hold byte-range shards of
one N-GiB stream with a 47-byte halo) plus an edited version of it (100 sparse
inserts/deletes/overwrites, synthgen.edited seed 3+rank).  Paper parameters: P = LBFS
(deg 63), w = 48, D = 8192, r = 0x78, bounds off.

One step = chunk both versions (all rows of SURVEY §8(a) that are active at the paper's
defaults: staging, rolling fingerprint, marker test, ordered compaction; at N > 1 the
per-rank candidate counts are exchanged with an NCCL all-gather).  Inputs are resident in HBM
and larger than L2 (no flush needed).  `value` = all ranks' input bytes / max-over-ranks device
time (CUDA events).  `e2e` = the same metric through the C ABI's host-fed mode: pinned host
buffers -> shred_feed (async H2D on the ctx's copy stream, double-buffered device slots) ->
shred_flush -> D2H of the cut offsets, all inside the timed region.

N > 1 (torchrun, one rank per GPU): configs[3] as strong scaling (BASELINE.json: "64 GiB random
stream byte-range sharded with halo across 1/2/4/8 B200").  The 2^36-byte stream (SplitMix64
seed 5) is split into N byte ranges at 4 KiB-aligned starts; each rank generates its range and
the 47 bytes before it on its GPU (untimed).  One step = dist.chunk_sharded on every rank (the
shard's candidates + the C2 count all-gather over NCCL; no host synchronisation), timed with
CUDA events, max over ranks.  `value` = 2^36 B / max-rank time per step.  `t1_ms` = the same
stream chunked whole on rank 0's GPU alone (the N = 1 time of this workload).  `--weak` keeps the
round-1 weak-scaling mode (configs[1] per rank).  N = 1 also reports `config3_64gib` (the whole
stream on one GPU) beside the configs[1] headline.

--impl reference: the CPU oracle (oracle/, R2 direct per-window reduction, all host cores) on
a bounded sample of the same workload per step; rank 0 only.
"""
from __future__ import annotations

import argparse
import json
import os
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

GiB = 1 << 30
METRIC = "chunking GB/s at 1/2/4/8 B200, device-resident & host-fed; % of HBM peak"
W = 48


def env_int(k, d):
    try:
        return int(os.environ.get(k, d))
    except ValueError:
        return d


def peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            p = json.load(f)
        return float(p["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs, copy test)"
    except Exception:
        return 6650.0, "fallback (B200_PROFILING.md 6.65 TB/s)"


def config(n_gpus, per_rank_bytes):
    return {"workload": "configs[1]: 1 GiB SplitMix64 file + edited version (100 sparse edits) per GPU, "
                        "device-resident; ranks hold byte-range shards of one stream with a 47-B halo",
            "params": "P=0xbfe6b8a5bf378d83 (deg 63), w=48, D=8192, r=0x78, min=0, max=inf",
            "bytes_per_step_per_gpu": per_rank_bytes,
            "l2": "inputs (1 GiB each) larger than the 126 MB L2; no flush",
            "parallelism": f"byte-range shards x{n_gpus}, count all-gather (NCCL)" if n_gpus > 1 else "1 GPU"}


STREAM3 = 1 << 36          # configs[3]: 64 GiB


def config3(n_gpus):
    return {"workload": "configs[3]: 64 GiB (2^36 B) SplitMix64 stream (seed 5), byte-range sharded with a "
                        "47-B halo across the ranks (4 KiB-aligned starts), device-resident",
            "params": "P=0xbfe6b8a5bf378d83 (deg 63), w=48, D=8192, r=0x78, min=0, max=inf",
            "bytes_per_step": STREAM3, "bytes_per_step_per_gpu": STREAM3 // n_gpus,
            "l2": "shards (>= 8 GiB) larger than the 126 MB L2; no flush",
            "parallelism": f"byte-range shards x{n_gpus}, C2 count all-gather (NCCL)"}


# ------------------------------------------------------------------------------- clocks (NVML)
class ClockSampler:
    REASONS = {0x4: "sw_power_cap", 0x8: "hw_slowdown", 0x20: "sw_thermal_slowdown",
               0x40: "hw_thermal_slowdown", 0x80: "hw_power_brake_slowdown", 0x2: "applications_clocks",
               0x1: "gpu_idle", 0x10: "sync_boost", 0x100: "display_clocks"}

    def __init__(self, dev_index):
        self.ok = False
        self.samples, self.reasons = [], 0
        try:
            import pynvml
            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(dev_index)
            self.max = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
            self.ok = True
        except Exception:
            pass
        self._stop = threading.Event()

    def _run(self):
        nv = self.nv
        get_r = getattr(nv, "nvmlDeviceGetCurrentClocksEventReasons", None) or \
            nv.nvmlDeviceGetCurrentClocksThrottleReasons
        k = 0
        while not self._stop.is_set():
            try:
                self.samples.append(nv.nvmlDeviceGetClockInfo(self.h, nv.NVML_CLOCK_SM))
                if k % 4 == 0:                 # the reasons query is the slower call on some boxes
                    self.reasons |= int(get_r(self.h))
            except Exception:
                pass
            k += 1
            time.sleep(0.0005)

    def __enter__(self):
        if self.ok:
            # the timed region can be ~20 ms: with the default 5 ms GIL switch interval the
            # sampler thread got as few as 1 sample in it, so switch threads every 0.1 ms meanwhile
            self._swi = sys.getswitchinterval()
            sys.setswitchinterval(1e-4)
            self.t = threading.Thread(target=self._run, daemon=True)
            self.t.start()
        return self

    def __exit__(self, *a):
        if self.ok:
            self._stop.set()
            self.t.join()
            sys.setswitchinterval(self._swi)

    def result(self):
        if not self.ok or not self.samples:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["nvml unavailable"]}
        return {"sm_mhz": float(np.median(self.samples)), "sm_max_mhz": float(self.max),
                "samples": len(self.samples),
                "reasons": [n for b, n in self.REASONS.items() if self.reasons & b and b != 0x1]}


# ------------------------------------------------------------------------------- CPU oracle timing
def oracle_rate(sample: np.ndarray, threads: int):
    import oracle
    t = time.perf_counter()
    c = oracle.candidates(sample, oracle.Params(), method=2, threads=threads)
    dt = time.perf_counter() - t
    return sample.size / dt / 1e9, dt, c.size


def cpu_model() -> str:
    try:
        with open("/proc/cpuinfo") as f:
            for ln in f:
                if ln.startswith("model name"):
                    return ln.split(":", 1)[1].strip()
    except OSError:
        pass
    return "unknown"


def oracle_samples(world: int, cores: int):
    """The bounded sample both arms time the oracle on (so that the main arm's cpu_baseline and
    the reference arm measure the same thing): slices of n <= 256 MiB, sized to ~2 s of oracle work
    on this host. N = 1: the configs[1] base file's first n bytes and its edited version
    (alternating); N > 1: consecutive slices of the configs[3] stream (seed 5)."""
    import synthgen
    cal = synthgen.random_bytes_fast(2, 8 << 20)
    rate, _, _ = oracle_rate(cal, cores)                   # calibration (also warms the tables)
    n = int(min(256 << 20, max(8 << 20, rate * 1e9 * 2.0)))
    n -= n % 4096
    if world == 1:
        base = synthgen.random_bytes_fast(2, n)
        ed, _ = synthgen.edited(base, 3, n_edits=max(1, min(100, n // (1 << 20))), min_gap=8192)
        return n, [base, ed]
    return n, [synthgen.random_bytes_fast(5, n, 0), synthgen.random_bytes_fast(5, n, n)]


def oracle_steps(samples, steps: int, cores: int):
    """Time `steps` oracle calls over the alternating samples; returns (total bytes, seconds,
    per-step GB/s)."""
    import oracle
    tot, per = 0, []
    t0 = time.perf_counter()
    for i in range(steps):
        s = samples[i % len(samples)]
        t = time.perf_counter()
        oracle.candidates(s, oracle.Params(), 2, cores)
        per.append(s.size / (time.perf_counter() - t) / 1e9)
        tot += s.size
    return tot, time.perf_counter() - t0, per


def cpu_measurements(runs: int = 5) -> dict:
    """The host-core baselines, measured in a FRESH process with no CUDA context (bench.py
    --cpu-only, started before the parent touches the GPU): the oracle (R2, all cores) on the same
    bounded sample and with the same timing code as the reference arm (`oracle_samples`,
    `oracle_steps`; round 1 timed it in-process after the CUDA work at half the rate, and early
    round 2 on a different sample), and the paper's §5.1 multithreaded rolling chunker
    on the whole 1 GiB base file."""
    import oracle
    import synthgen
    oracle.build()
    cores = sorted(os.sched_getaffinity(0))
    nc = len(cores)
    n, samples = oracle_samples(1, nc)
    oracle_steps(samples, 3, nc)                            # warm-up steps (the reference arm: W >= 3)
    tot, dt, per = oracle_steps(samples, 2 * runs, nc)
    rate1, dt1, _ = oracle_rate(samples[0][: 8 << 20], 1)
    out = {"cpu_baseline": {
        "value": round(tot / dt / 1e9, 4), "unit": "GB/s", "cores": nc, "kind": "oracle",
        "sample": f"{2 * runs} steps of {n / 2**20:.0f} MiB, alternating the configs[1] base file's first "
                  f"{n / 2**20:.0f} MiB (SplitMix64 seed 2) and its edited version, R2 direct per-window "
                  f"reduction (48 table lookups/window), {nc} threads, fresh process without a CUDA "
                  f"context; the reference arm's sample and timing code",
        "runs": [round(r, 4) for r in per], "median_step": round(float(np.median(per)), 4),
        "affinity": f"cpus {cores[0]}-{cores[-1]} ({nc})",
        "value_1core": round(rate1, 4), "sample_1core": f"first 8 MiB, 1 thread, {dt1:.1f} s",
        "cpu_model": cpu_model()}}
    host = synthgen.random_bytes_fast(2, GiB)             # = the device's synth_fill(seed 2)
    try:
        import cpu_baseline as cb
        cb.build()
        cb.chunk(host[: 64 << 20], threads=nc)
        cr, cnt = [], 0
        for _ in range(runs):
            t0 = time.perf_counter()
            cnt = int(cb.chunk(host, threads=nc).size)
            cr.append(host.size / (time.perf_counter() - t0) / 1e9)
        out["cpu_chunker"] = {"value": round(float(np.median(cr)), 3), "unit": "GB/s", "cores": nc,
                              "runs": [round(r, 3) for r in cr], "count": cnt,
                              "kind": "multithreaded rolling chunker (PAPER.md §5.1 SPMD, gcc -O3 -march=x86-64-v3)",
                              "sample": f"the whole 1 GiB base file, median of {runs} runs, fresh process"}
    except Exception as e:
        out["cpu_chunker"] = {"error": repr(e)}
    return out


def cpu_measurements_subprocess() -> dict:
    import subprocess
    r = subprocess.run([sys.executable, os.path.abspath(__file__), "--cpu-only"], capture_output=True, text=True)
    for ln in reversed(r.stdout.splitlines()):
        if ln.startswith("{"):
            return json.loads(ln)
    return {"cpu_baseline": {"error": (r.stderr or r.stdout)[-400:]}}


# ------------------------------------------------------------------------------- reference arm
def run_reference(args, rank, world):
    if rank != 0:
        return
    import oracle
    import synthgen
    oracle.build()
    cores = len(os.sched_getaffinity(0))
    per_rank = 2 * GiB
    # each step: a bounded sample of the workload (oracle_samples; the main arm's cpu_baseline
    # times the same sample with the same code)
    n, samples = oracle_samples(world, cores)
    oracle_steps(samples, args.warmup, cores)
    tot, dt, _ = oracle_steps(samples, args.steps, cores)
    v = tot / dt / 1e9
    line = {"metric": METRIC, "value": round(v, 4), "unit": "GB/s", "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": round(dt / args.steps * 1e3, 3), "higher_is_better": True,
            "scaling": "weak" if world == 1 else "strong", "vs_baseline": None, "dtype": "u8", "data": "synthetic",
            "config": config(world, per_rank) if world == 1 else config3(world), "impl": "reference",
            "cpu_baseline": {"value": round(v, 4), "unit": "GB/s", "cores": cores, "kind": "oracle",
                             "sample": (f"each step = {n / 2**20:.0f} MiB of the base file or its edited "
                                        f"version (alternating)" if world == 1 else
                                        f"each step = {n / 2**20:.0f} MiB of the configs[3] stream (seed 5)")
                                       + f", R2 oracle, {cores} threads"},
            "e2e": {"value": round(v, 4), "unit": "GB/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


# ------------------------------------------------------------------------------- N > 1: configs[3]
def run_scaled(args, rank, world, local):
    """configs[3] strong scaling (see the module docstring)."""
    import torch
    import torch.distributed as dist
    import paper_conf_fast_bhatotiarv12_b200 as pkg
    from paper_conf_fast_bhatotiarv12_b200 import dist as sd

    backend = os.environ.get("SHRED_BENCH_BACKEND", "nccl")        # test-only override (gloo)
    local = int(os.environ.get("SHRED_BENCH_DEVICE", local))
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if backend == "nccl":
        dist.init_process_group("nccl", device_id=dev)
    else:
        dist.init_process_group(backend)
    total = int(os.environ.get("SHRED_BENCH_STREAM", STREAM3))     # test-only override of 2^36
    start, end = sd.shard_bounds(total, world, rank)
    halo = sd.halo_of(start)
    x = torch.empty(end - start + halo, dtype=torch.uint8, device=dev)
    pkg.synth_fill(x, 5, start - halo)                              # untimed: shard + halo on device
    ch = pkg.Chunker(pkg.Params(), device=local)
    cap = sd._expected_cap(ch, end - start)
    stream = torch.cuda.current_stream()

    def maxr(v):                                                     # max over ranks of a float
        t = torch.tensor([v], dtype=torch.float64, device=dev)
        if backend != "nccl":
            t = t.cpu()
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        return float(t.item())

    for _ in range(args.warmup):
        res = sd.chunk_sharded(x, halo, start, total, ch, cap=cap)
    torch.cuda.synchronize()
    n_total = res.total                                             # (synchronises; outside timing)
    assert res.local.numel() == int(res.counts[rank])
    dist.barrier()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    l0 = ch.launches
    ch.profile(True)
    with ClockSampler(local) as clk:
        e0.record(stream)
        for _ in range(args.steps):
            sd.chunk_sharded(x, halo, start, total, ch, cap=cap)
        e1.record(stream)
        torch.cuda.synchronize()
    ch.profile(False)
    launches = ch.launches - l0
    k_ms, k_n, k_bytes = ch.profile_read()
    ms = maxr(e0.elapsed_time(e1))
    value = total * args.steps / (ms * 1e-3) / 1e9
    hbm, hbm_src = peaks()
    k_avg = k_ms / max(1, k_n)
    achieved = (k_bytes / max(1, k_n)) / (k_avg * 1e-3) / 1e9 if k_n else None
    line = {"metric": METRIC, "value": round(value, 2), "unit": "GB/s", "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": round(ms / args.steps, 4), "higher_is_better": True,
            "scaling": "strong", "vs_baseline": None, "dtype": "u8", "data": "synthetic",
            "config": config3(world), "hbm_frac": round(value / world / hbm, 4),
            "tG_ms": round(ms / args.steps, 4), "candidates_total": n_total,
            "roofline": {"bound": "hbm", "achieved": round(achieved, 1) if achieved else None, "peak": hbm,
                         "unit": "GB/s", "frac": round(achieved / hbm, 4) if achieved else None, "traffic": None,
                         "kernel": "k1_bulk<K63> (rank 0)", "launches": k_n, "avg_launch_ms": round(k_avg, 4),
                         "peak_source": hbm_src},
            "clocks": clk.result(), "gpu_launches": launches}
    try:
        with open(os.path.join(ROOT, "tests", "golden", "oracle_fullsize.json")) as f:
            g = json.load(f)["configs3"]
        if g["n"] == total:
            line["matches_oracle_count"] = n_total == g["candidates"]["count"]
    except Exception:
        pass
    # bounded mode (min 2048 / max 65536) with the distributed size rule ("chain") as a side line
    if not args.no_extra:
        chb = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536), device=local)
        rb = sd.chunk_sharded(x, halo, start, total, chb, cap=cap)
        torch.cuda.synchronize()
        dist.barrier()
        b0, b1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        b0.record(stream)
        for _ in range(max(2, args.steps // 4)):
            rb = sd.chunk_sharded(x, halo, start, total, chb, cap=cap)
        b1.record(stream)
        torch.cuda.synchronize()
        bms = maxr(b0.elapsed_time(b1)) / max(2, args.steps // 4)
        line["bounded_2048_65536"] = {"value": round(total / (bms * 1e-3) / 1e9, 2), "unit": "GB/s",
                                      "rounds": rb.rounds, "mode": "chain (distributed size rule)",
                                      "note": "includes one host synchronisation per step (the chain's convergence check)"}
        del chb
    # e2e: every rank feeds (a bounded sample of) its shard from pinned host memory through the
    # C ABI (shred_feed + shred_flush + D2H of the cuts); aggregate bytes / max-rank time
    if not args.no_e2e:
        import synthgen
        m = min(end - start, 2 * GiB)
        pin = torch.empty(m, dtype=torch.uint8).pin_memory()
        synthgen.fill_fast(pin.numpy(), 5, start, threads=max(1, len(os.sched_getaffinity(0)) // world))
        che = pkg.Chunker(pkg.Params(), device=local)
        che.set_ring(2, 256 << 20)
        ecap = m // 2048 + 65536
        eo = torch.empty(ecap, dtype=torch.int64, device=dev)
        en = torch.zeros(1, dtype=torch.int64, device=dev)
        en_h = torch.zeros(1, dtype=torch.int64).pin_memory()
        res_h = torch.empty(ecap, dtype=torch.int64).pin_memory()
        fo = torch.empty(1, dtype=torch.int64, device=dev)
        fn = torch.zeros(1, dtype=torch.int64, device=dev)

        def e2e_step():
            che.feed_async(pin, eo, en)
            pkg.lib().shred_flush(che._ctx, fo.data_ptr(), 1, fn.data_ptr(), stream.cuda_stream)
            en_h.copy_(en, non_blocking=True)
            stream.synchronize()
            a = int(en_h[0])
            res_h[:a].copy_(eo[:a], non_blocking=True)
            return a

        for _ in range(2):
            e2e_step()
        torch.cuda.synchronize()
        dist.barrier()
        s0, s1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        s0.record(stream)
        es = max(2, args.steps // 4)
        for _ in range(es):
            a = e2e_step()
        s1.record(stream)
        torch.cuda.synchronize()
        ems = maxr(s0.elapsed_time(s1))
        line["e2e"] = {"value": round(world * m * es / (ems * 1e-3) / 1e9, 3), "unit": "GB/s",
                       "h2d_bytes_per_step": m, "d2h_bytes_per_step": 8 * a + 8,
                       "sample": f"each rank feeds the first {m / 2**30:.2f} GiB of its shard from pinned host memory",
                       "api": "shred_feed(pinned host, 2 x 256 MiB device slots) + shred_flush + D2H of cuts"}
        del pin, che
    # t1: the whole stream on rank 0's GPU alone (same call path, one shard = the stream)
    dist.barrier()
    if rank == 0 and not args.no_extra:
        try:
            del x
            torch.cuda.empty_cache()
            xx = torch.empty(total, dtype=torch.uint8, device=dev)
            pkg.synth_fill(xx, 5, 0)
            o1 = torch.empty(sd._expected_cap(ch, total), dtype=torch.int64, device=dev)
            n1 = torch.zeros(1, dtype=torch.int64, device=dev)
            for _ in range(2):
                ch.candidates_range_async(xx, 0, 0, total, o1, n1)
            torch.cuda.synchronize()
            t0_, t1_ = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            t0_.record(stream)
            for _ in range(3):
                ch.candidates_range_async(xx, 0, 0, total, o1, n1)
            t1_.record(stream)
            torch.cuda.synchronize()
            line["t1_ms"] = round(t0_.elapsed_time(t1_) / 3, 4)
            line["t1_candidates"] = int(n1.item())
            del xx
        except Exception as e:
            line["t1_ms"] = None
            line["t1_error"] = repr(e)
    dist.barrier()
    if rank == 0:
        print(json.dumps(line), flush=True)
    dist.destroy_process_group()


# ------------------------------------------------------------------------------- our arm
def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=5)
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--no-extra", action="store_true", help="skip the bounded / k32 side measurements")
    ap.add_argument("--cpu-only", action="store_true", help=argparse.SUPPRESS)   # internal: fresh-process CPU leg
    ap.add_argument("--weak", action="store_true", help="N > 1: round-1 weak scaling (configs[1] per rank)")
    ap.add_argument("--variant", default="paper", choices=["paper", "k32", "k32t"],
                    help="profiling aid: k32 = P 0x104C11DB7, k32t = x^31+x^13+1 on the main path (not the headline)")
    args = ap.parse_args()
    args.warmup = max(3, args.warmup)

    rank, world, local = env_int("RANK", 0), env_int("WORLD_SIZE", 1), env_int("LOCAL_RANK", 0)
    if args.cpu_only:
        print(json.dumps(cpu_measurements()), flush=True)
        return
    if args.impl == "reference":
        return run_reference(args, rank, world)
    if world > 1 and not args.weak:
        return run_scaled(args, rank, world, local)
    # host-core baselines first, in a fresh process, before this process creates a CUDA context
    cpu = cpu_measurements_subprocess() if (not args.no_cpu and rank == 0 and world == 1) else None

    import torch
    import torch.distributed as dist
    import synthgen
    import paper_conf_fast_bhatotiarv12_b200 as pkg

    # Test-only overrides (exercise the N > 1 code path on a 1-GPU box): SHRED_BENCH_BACKEND=gloo
    # and SHRED_BENCH_DEVICE=0 put every rank on one device.  Real runs: NCCL, one GPU per rank.
    backend = os.environ.get("SHRED_BENCH_BACKEND", "nccl")
    local = int(os.environ.get("SHRED_BENCH_DEVICE", local))
    torch.cuda.set_device(local)
    if world > 1:
        if backend == "nccl":
            dist.init_process_group("nccl", device_id=torch.device("cuda", local))
        else:
            dist.init_process_group(backend)
    dev = torch.device("cuda", local)

    def coll_dev(t):            # gloo exchanges host tensors
        return t if backend == "nccl" else t.cpu()
    stream = torch.cuda.current_stream()

    # ---- inputs (untimed): this rank's shard of stream seed 2 with its halo, and an edited file
    halo = min(W - 1, rank * GiB)
    base_h = torch.empty(GiB + halo, dtype=torch.uint8, device=dev)
    pkg.synth_fill(base_h, 2, rank * GiB - halo)
    base = base_h[halo:]
    host_base = base.cpu().numpy()
    ed_np, _ = synthgen.edited(host_base, 3 + rank)
    edited = torch.from_numpy(ed_np).to(dev)
    per_rank_bytes = int(base.numel() + edited.numel())

    main_params = pkg.Params(poly={"paper": pkg.Params().poly, "k32": 0x104C11DB7, "k32t": 0x80002001}[args.variant])
    ch = pkg.Chunker(main_params, device=local)
    cap = GiB // 2048 + 65536
    out0 = torch.empty(cap, dtype=torch.int64, device=dev)
    out1 = torch.empty(cap, dtype=torch.int64, device=dev)
    n0 = torch.zeros(1, dtype=torch.int64, device=dev)
    n1 = torch.zeros(1, dtype=torch.int64, device=dev)
    counts = torch.zeros(world, dtype=torch.int64, device=dev)
    total = world * GiB

    def step():
        if world == 1:
            ch.chunk_async(base, out0, n0)
        else:
            rc = pkg.lib().shred_candidates_range(ch._ctx, base_h.data_ptr(), halo, rank * GiB, GiB, total,
                                                  out0.data_ptr(), cap, n0.data_ptr(), stream.cuda_stream)
            ch._check(rc, "shred_candidates_range")
        ch.chunk_async(edited, out1, n1)
        if world > 1:
            if backend == "nccl":
                dist.all_gather_into_tensor(counts, n0)   # C2: per-rank candidate counts
            else:
                cc = torch.zeros(world, dtype=torch.int64)
                dist.all_gather_into_tensor(cc, n0.cpu())
                counts.copy_(cc)

    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    l0 = ch.launches
    ch.profile(True)
    with ClockSampler(local) as clk:
        e0.record(stream)
        for _ in range(args.steps):
            step()
        e1.record(stream)
        torch.cuda.synchronize()
    ch.profile(False)
    launches = ch.launches - l0
    k_ms, k_n, k_bytes = ch.profile_read()
    if world > 1:
        dist.barrier()
    ms = e0.elapsed_time(e1)
    t = coll_dev(torch.tensor([ms], dtype=torch.float64, device=dev))
    if world > 1:
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
    ms_max = float(t.item())
    value = world * per_rank_bytes * args.steps / (ms_max * 1e-3) / 1e9
    n_cand = int(n0.item())
    assert n_cand <= cap and int(n1.item()) <= cap
    hbm, hbm_src = peaks()

    # ---- roofline of the hot kernel (k1_bulk), live CUDA events on the launching stream
    k_avg_ms = k_ms / max(1, k_n)
    k_bytes_per_launch = k_bytes / max(1, k_n)
    achieved = k_bytes_per_launch / (k_avg_ms * 1e-3) / 1e9 if k_n else None
    traffic, traffic_src = None, None
    try:
        with open(os.path.join(ROOT, "profiles", "k1_traffic.json")) as f:
            tr = json.load(f)
        traffic = tr.get("dram_bytes_per_launch")
        traffic_src = tr.get("source")
    except Exception:
        pass
    roofline = {"bound": "hbm", "achieved": round(achieved, 1) if achieved else None, "peak": hbm,
                "unit": "GB/s", "frac": round(achieved / hbm, 4) if achieved else None, "traffic": traffic,
                "kernel": f"k1_bulk<{ch.path.upper()}>", "launches": k_n, "avg_launch_ms": round(k_avg_ms, 4),
                "algorithmic_bytes_per_launch": int(k_bytes_per_launch),
                "share_of_step": round(k_ms / ms, 4) if ms else None, "peak_source": hbm_src,
                "traffic_source": traffic_src,
                "note": "algorithmic bytes = 1 B read per input byte (+8 B per candidate, ~0.001 B/B); "
                        "the kernel is bound by the shared-memory lookup datapath below HBM (DESIGN.md)"}
    # the unit that actually binds: 128 B/clk/SM of shared-memory datapath; per input byte the K63
    # loop moves 16 B of table lookups + 1 B TMA write + 1 B LDS read (K32: 8 + 1 + 1)
    smem_bpb = 18.0 if ch.path == "k63" else 10.0
    clk_mhz = clk.result().get("sm_mhz") or 1965.0
    nsm = torch.cuda.get_device_properties(dev).multi_processor_count
    smem_ceiling = nsm * clk_mhz * 1e6 * 128.0 / smem_bpb / 1e9
    if achieved:
        roofline["smem_datapath"] = {"ceiling_gbs": round(smem_ceiling, 1), "frac": round(achieved / smem_ceiling, 4),
                                     "bytes_per_input_byte": smem_bpb, "sms": nsm, "sm_mhz": clk_mhz,
                                     "source": "128 B/clk/SM SMEM/L1 data path (B300_MICROARCH.md); ncu "
                                               f"l1tex__data_pipe_lsu_wavefronts in {traffic_src}"}

    line = {"metric": METRIC, "value": round(value, 2), "unit": "GB/s", "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": round(ms_max / args.steps, 4), "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "u8", "data": "synthetic",
            "config": config(world, per_rank_bytes), "hbm_frac": round(value / world / hbm, 4),
            "roofline": roofline, "clocks": clk.result(), "gpu_launches": launches,
            "candidates_rank0": n_cand,
            "paper_context": {"note": "PAPER.md numbers on other hardware: context only, not a target",
                              "gpu": "full Shredder <= 2.5 GB/s (Fig. 12 axis, L1016-L1037), Tesla C2050 "
                                     "(Fermi, 144 GB/s GDDR5), CUDA 4.0",
                              "gpu_device_time": "16-256 MB buffers in 11.39-171.4 ms = 1.47-1.57 GB/s (Table 2, L766-L770)",
                              "cpu_ratio": "GPU > 5x the 12-thread pthreads chunker on 2x Xeon X5650 (L88-L90, L1100-L1102)"}}

    # ---- e2e: host-fed through the C ABI (pinned host -> shred_feed -> flush -> D2H)
    if not args.no_e2e:
        pin_base = torch.empty(base.numel(), dtype=torch.uint8).pin_memory()
        pin_base.copy_(base.cpu())
        pin_ed = torch.from_numpy(ed_np).pin_memory()
        che = pkg.Chunker(pkg.Params(), device=local)
        che.set_ring(2, 256 << 20)
        ecap = GiB // 2048 + 65536
        eo = torch.empty(ecap, dtype=torch.int64, device=dev)
        en = torch.zeros(2, dtype=torch.int64, device=dev)
        en_h = torch.zeros(2, dtype=torch.int64).pin_memory()
        res_h = torch.empty(2 * ecap, dtype=torch.int64).pin_memory()
        fo = torch.empty(1, dtype=torch.int64, device=dev)
        fn = torch.zeros(1, dtype=torch.int64, device=dev)
        d2h = [0]

        def e2e_step():
            che.feed_async(pin_base, eo, en[0:1])
            pkg.lib().shred_flush(che._ctx, fo.data_ptr(), 1, fn.data_ptr(), stream.cuda_stream)
            en_h.copy_(en, non_blocking=True)
            stream.synchronize()
            a = int(en_h[0])
            res_h[:a].copy_(eo[:a], non_blocking=True)
            che.feed_async(pin_ed, eo, en[1:2])
            pkg.lib().shred_flush(che._ctx, fo.data_ptr(), 1, fn.data_ptr(), stream.cuda_stream)
            en_h.copy_(en, non_blocking=True)
            stream.synchronize()
            b = int(en_h[1])
            res_h[a:a + b].copy_(eo[:b], non_blocking=True)
            d2h[0] = 8 * (a + b) + 16
            return a, b

        for _ in range(max(2, args.warmup)):
            e2e_step()
        torch.cuda.synchronize()
        if world > 1:
            dist.barrier()
        s0, s1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        s0.record(stream)
        for _ in range(args.steps):
            a, b = e2e_step()
        s1.record(stream)
        torch.cuda.synchronize()
        ems = s0.elapsed_time(s1)
        # the last e2e step's offsets (base + edited, copied back to pinned host) == the
        # device-resident path's, element by element (world 1: both chunk the same two files)
        match = None
        if world == 1:
            na_, nb_ = int(n0.item()), int(n1.item())
            match = bool(a == na_ and b == nb_ and torch.equal(res_h[:a], out0[:na_].cpu())
                         and torch.equal(res_h[a:a + b], out1[:nb_].cpu()))
        et = coll_dev(torch.tensor([ems], dtype=torch.float64, device=dev))
        if world > 1:
            dist.all_reduce(et, op=dist.ReduceOp.MAX)
        ems = float(et.item())
        ev = world * per_rank_bytes * args.steps / (ems * 1e-3) / 1e9
        # H2D peak on this box for context (256 MiB pinned copy, best of 5)
        tmp = torch.empty(256 << 20, dtype=torch.uint8, device=dev)
        best = 1e9
        for _ in range(5):
            q0, q1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            q0.record(stream)
            tmp.copy_(pin_base[: 256 << 20], non_blocking=True)
            q1.record(stream)
            torch.cuda.synchronize()
            best = min(best, q0.elapsed_time(q1))
        h2d_peak = (256 << 20) / (best * 1e-3) / 1e9
        # ring depth 3 (the paper's Fig. 9 pipeline-depth analogue), same step
        che.set_ring(3, 256 << 20)
        e2e_step()
        torch.cuda.synchronize()
        r0, r1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        r0.record(stream)
        for _ in range(max(2, args.steps // 2)):
            e2e_step()
        r1.record(stream)
        torch.cuda.synchronize()
        ev3 = world * per_rank_bytes * max(2, args.steps // 2) / (r0.elapsed_time(r1) * 1e-3) / 1e9
        line["e2e"] = {"value": round(ev, 3), "unit": "GB/s", "h2d_bytes_per_step": per_rank_bytes,
                       "ring3_value": round(ev3, 3),
                       "d2h_bytes_per_step": d2h[0], "ms_per_step": round(ems / args.steps, 3),
                       "api": "shred_feed(pinned host, 2 x 256 MiB device slots) + shred_flush + D2H of cuts",
                       "h2d_peak_gbs": round(h2d_peak, 2), "frac_of_h2d_peak": round(ev / world / h2d_peak, 4),
                       "cuts_match_device_path": match}
        del tmp

    # ---- side measurements (not the headline): bounded mode and the k32 instantiation
    if not args.no_extra and world == 1:
        def timed(chx, x, reps=5):
            o = torch.empty(cap, dtype=torch.int64, device=dev)
            nn = torch.zeros(1, dtype=torch.int64, device=dev)
            chx.chunk_async(x, o, nn)
            torch.cuda.synchronize()
            a0, a1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            a0.record(stream)
            for _ in range(reps):
                chx.chunk_async(x, o, nn)
            a1.record(stream)
            torch.cuda.synchronize()
            return x.numel() * reps / (a0.elapsed_time(a1) * 1e-3) / 1e9
        try:
            chb = pkg.Chunker(pkg.Params(min_size=2048, max_size=65536), device=local)
            line["bounded_2048_65536"] = {"value": round(timed(chb, base), 2), "unit": "GB/s",
                                          "note": "size rule on: parallel speculative size-rule kernels (sb_*), no host sync"}
            # min >= D: the speculative blocks rarely re-sync; the repair passes take over
            bd = {}
            for mn, mx in ((8192, 65536), (65536, 0)):
                chx = pkg.Chunker(pkg.Params(min_size=mn, max_size=mx), device=local)
                bd[f"min{mn}_max{mx}"] = round(timed(chx, base, reps=3), 2)
                del chx
            line["bounded_2048_65536"]["min_ge_D"] = bd
            c32 = pkg.Chunker(pkg.Params(poly=0x104C11DB7), device=local)
            v32 = timed(c32, base)
            line["k32_variant"] = {"value": round(v32, 2), "unit": "GB/s", "hbm_frac": round(v32 / hbm, 4),
                                   "params": "P=0x104C11DB7 (deg 32, irreducible), other params as paper",
                                   "mode": c32.mode}
            # the multiply-reduction u32 kernel (MODE_K32T): an irreducible trinomial whose top-byte
            # reduction is one integer product (no T lookup); ALU-bound (profiles/r02_k32_ab.txt)
            c3t = pkg.Chunker(pkg.Params(poly=0x80002001), device=local)
            v3t = timed(c3t, base)
            line["k32t_variant"] = {"value": round(v3t, 2), "unit": "GB/s", "hbm_frac": round(v3t / hbm, 4),
                                    "params": "P=x^31+x^13+1 (0x80002001, irreducible trinomial), other params as paper",
                                    "mode": c3t.mode}
            del c3t
            # the u64-state analogue (MODE_K63T) for a sparse degree-63 polynomial
            c6t = pkg.Chunker(pkg.Params(poly=0x8000000000000801), device=local)
            v6t = timed(c6t, base)
            line["k63t_variant"] = {"value": round(v6t, 2), "unit": "GB/s", "hbm_frac": round(v6t / hbm, 4),
                                    "params": "P=x^63+x^11+1 (0x8000000000000801, irreducible trinomial), other params as paper",
                                    "mode": c6t.mode}
            del c6t
            # long windows (w > 64): the hot kernel with the pops from a second TMA tile
            lw = {}
            for wv in (128, 1000):
                clw = pkg.Chunker(pkg.Params(window=wv), device=local)
                lw[f"w{wv}"] = round(timed(clw, base), 2)
                del clw
            line["long_window_variant"] = {"value": lw["w128"], "unit": "GB/s", "w1000": lw["w1000"],
                                           "params": "w = 128 (and 1000), other params as paper",
                                           "note": "windows 65-4096 on k1_bulk: pops from a second TMA tile "
                                                   "(DESIGN.md §5 Long windows)"}
            # content sensitivity. Text-like bytes (words from a fixed
            # 1,000-word list; skewed outgoing bytes for the U lookups), 64 MiB generated on the
            # host and tiled to 256 MiB on the device; paper params on the same ctx.
            import synthgen
            tl = torch.from_numpy(synthgen.text_like(7, 64 << 20)).to(dev).repeat(4)
            vt = timed(ch, tl)
            vr = timed(ch, base[: 256 << 20])
            line["text_like_256mib"] = {"value": round(vt, 2), "unit": "GB/s", "hbm_frac": round(vt / hbm, 4),
                                        "random_256mib": round(vr, 2),
                                        "note": "words from a 1,000-word list (64 MiB tiled x4), paper params; "
                                                "random_256mib: the first 256 MiB of the random file, same call"}
            del tl
            # configs[0]: 1 MiB per call, launch-latency bound -> report microseconds per call
            small = base[: 1 << 20]
            o_s = torch.empty(4096, dtype=torch.int64, device=dev)
            n_s = torch.zeros(1, dtype=torch.int64, device=dev)

            def small_latency(chx):
                # warm-up long enough (~10 ms of back-to-back calls) for the SM clock to settle
                # after the host-side phases above; a short burst can run below the boost clock
                for _ in range(800):
                    chx.chunk_async(small, o_s, n_s)
                torch.cuda.synchronize()
                q0, q1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                q0.record(stream)
                for _ in range(1000):
                    chx.chunk_async(small, o_s, n_s)
                q1.record(stream)
                torch.cuda.synchronize()
                us = q0.elapsed_time(q1) * 1e3 / 1000
                # the same call captured once into a CUDA graph and replayed (no per-call launches)
                gs = torch.cuda.Stream()
                gs.wait_stream(stream)
                with torch.cuda.stream(gs):
                    chx.chunk_async(small, o_s, n_s, stream=gs)
                torch.cuda.synchronize()
                cg = torch.cuda.CUDAGraph()
                with torch.cuda.graph(cg, stream=gs):
                    for _ in range(20):                  # 20 calls per graph: no per-call launch cost
                        chx.chunk_async(small, o_s, n_s, stream=gs)
                cg.replay()
                torch.cuda.synchronize()
                for _ in range(20):
                    cg.replay()
                q0.record(stream)
                for _ in range(50):
                    cg.replay()
                q1.record(stream)
                torch.cuda.synchronize()
                return us, q0.elapsed_time(q1) * 1e3 / 1000, int(n_s.item())

            us_b, us_graph_b, n_b = small_latency(pkg.Chunker(pkg.Params(min_size=2048, max_size=65536), device=local))
            us, us_graph, n_small = small_latency(ch)
            line["config1_1mib"] = {"us_per_call": round(us, 2), "us_per_call_in_graph": round(us_graph, 2),
                                    "gbs": round((1 << 20) / (us * 1e-6) / 1e9, 1),
                                    "candidates": n_small,
                                    "bounded_us_per_call": round(us_b, 2),
                                    "bounded_us_per_call_in_graph": round(us_graph_b, 2), "bounded_cuts": n_b,
                                    "note": "configs[0] size, device-resident, back-to-back calls on one stream; "
                                            "bounded_*: the same call with the size rule on (min 2048 / max 65536)"}
            # f2: SHA-256 of every chunk.  One buffer alone is bound by its longest chunk (a
            # sequential hash on one lane); a batch of buffers shares one length-sorted work
            # list (shred_hash_chunks_batch), so the long chains overlap the other buffers' work.
            # Measured: the 1 GiB base file alone; 3 x the base file as one batch (3 digest
            # arrays); the step's two files (base + edited) chunked then hashed as one batch.
            digs = [torch.empty((cap + 1) * 32, dtype=torch.uint8, device=dev) for _ in range(3)]
            ch.chunk_async(base, out0, n0)
            ch.chunk_async(edited, out1, n1)
            ch.hash_chunks_async(base, out0, n0, digs[0])
            ch.hash_chunks_batch_async([(base, out0, n0, d) for d in digs])     # grows the work list once
            torch.cuda.synchronize()
            h0, h1, h2, h3 = (torch.cuda.Event(enable_timing=True) for _ in range(4))
            h0.record(stream)
            for _ in range(3):
                ch.hash_chunks_async(base, out0, n0, digs[0])
            h1.record(stream)
            for _ in range(3):
                ch.hash_chunks_batch_async([(base, out0, n0, d) for d in digs])
            h2.record(stream)
            for _ in range(3):
                ch.chunk_async(base, out0, n0)
                ch.chunk_async(edited, out1, n1)
                ch.hash_chunks_batch_async([(base, out0, n0, digs[0]), (edited, out1, n1, digs[1])])
            h3.record(stream)
            torch.cuda.synchronize()
            # the same on bounded chunks (min 2048 / max 65536): the longest chunk is capped
            ob = torch.empty(cap, dtype=torch.int64, device=dev)
            nb_ = torch.zeros(1, dtype=torch.int64, device=dev)
            chb.chunk_async(base, ob, nb_)
            chb.hash_chunks_async(base, ob, nb_, digs[2])
            torch.cuda.synchronize()
            g0, g1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            g0.record(stream)
            for _ in range(3):
                chb.hash_chunks_async(base, ob, nb_, digs[2])
            g1.record(stream)
            torch.cuda.synchronize()
            gbs = lambda nbytes, a, b: round(nbytes / (a.elapsed_time(b) * 1e-3) / 1e9, 2)   # noqa: E731
            line["hash_sha256"] = {"value": gbs(9 * base.numel(), h1, h2),
                                   "unit": "GB/s", "chunks_per_buffer": int(n0.item()) + 1,
                                   "single_buffer_value": gbs(3 * base.numel(), h0, h1),
                                   "bounded_chunks_value": gbs(3 * base.numel(), g0, g1),
                                   "chunk_plus_hash": gbs(3 * per_rank_bytes, h2, h3),
                                   "note": "SURVEY §8(f) f2: SHA-256 per chunk.  value: the 1 GiB base file x3 "
                                           "hashed as one batch (shred_hash_chunks_batch); single_buffer_value: "
                                           "one buffer per call (bound by its longest chunk); chunk_plus_hash: "
                                           "the step's two files chunked, then hashed as one batch, on the device"}
            del digs
            # configs[3] on one GPU: the whole 2^36-byte stream (seed 5) in one call; the N = 1
            # time of the strong-scaling workload that `bench.py --gpus N` runs at N > 1
            try:
                free, _ = torch.cuda.mem_get_info(dev)
                if free > STREAM3 + (8 << 30):
                    x3 = torch.empty(STREAM3, dtype=torch.uint8, device=dev)
                    pkg.synth_fill(x3, 5, 0)
                    o3 = torch.empty(STREAM3 // 4096 + 65536, dtype=torch.int64, device=dev)
                    n3 = torch.zeros(1, dtype=torch.int64, device=dev)
                    for _ in range(2):
                        ch.chunk_async(x3, o3, n3)
                    torch.cuda.synchronize()
                    q0.record(stream)
                    for _ in range(3):
                        ch.chunk_async(x3, o3, n3)
                    q1.record(stream)
                    torch.cuda.synchronize()
                    t3 = q0.elapsed_time(q1) / 3
                    c3 = {"ms": round(t3, 3), "value": round(STREAM3 / (t3 * 1e-3) / 1e9, 2), "unit": "GB/s",
                          "candidates": int(n3.item()),
                          "note": "configs[3] stream whole on 1 GPU (t1 of the N > 1 strong-scaling runs)"}
                    try:
                        with open(os.path.join(ROOT, "tests", "golden", "oracle_fullsize.json")) as f:
                            c3["matches_oracle_count"] = c3["candidates"] == json.load(f)["configs3"]["candidates"]["count"]
                    except Exception:
                        pass
                    line["config3_64gib"] = c3
                    del x3, o3
                    torch.cuda.empty_cache()
            except Exception as e:
                line["config3_64gib"] = {"error": repr(e)}
            # configs[2]: a 16 GiB stream (seed 4) in pinned host memory fed as 64 buffers of
            # 256 MiB through shred_feed (the window carry across buffers), 2- and 3-slot device
            # rings, then shred_flush; the count is checked against the stored oracle count
            try:
                import synthgen
                n2 = 1 << 34
                h2 = torch.empty(n2, dtype=torch.uint8).pin_memory()
                synthgen.fill_fast(h2.numpy(), 4)
                piece = 256 << 20
                c2 = {"unit": "GB/s", "feeds": n2 // piece, "feed_bytes": piece}
                try:
                    with open(os.path.join(ROOT, "tests", "golden", "oracle_fullsize.json")) as f:
                        oc2 = json.load(f)["configs2"]["candidates"]["count"]
                except Exception:
                    oc2 = None
                for slots in (2, 3):
                    cf = pkg.Chunker(pkg.Params(), device=local)
                    cf.set_ring(slots, piece)
                    fo2 = torch.empty((n2 // piece, 1 << 16), dtype=torch.int64, device=dev)
                    fn2 = torch.zeros(n2 // piece, dtype=torch.int64, device=dev)
                    for it in range(2):                    # the first pass allocates the ring
                        torch.cuda.synchronize()
                        a0, a1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                        a0.record(stream)
                        for j in range(n2 // piece):
                            cf.feed_async(h2[j * piece:(j + 1) * piece], fo2[j], fn2[j:j + 1])
                        tail = cf.flush()
                        a1.record(stream)
                        torch.cuda.synchronize()
                    cnt = int(fn2.sum().item()) + int(tail.numel())
                    c2[f"ring{slots}_value"] = round(n2 / (a0.elapsed_time(a1) * 1e-3) / 1e9, 2)
                    c2[f"ring{slots}_candidates"] = cnt
                    if oc2 is not None:
                        c2[f"ring{slots}_matches_oracle_count"] = cnt == oc2
                    del cf, fo2, fn2
                c2["value"] = max(c2["ring2_value"], c2["ring3_value"])
                c2["note"] = ("configs[2]: 16 GiB from pinned host memory, 64 x 256 MiB shred_feed + shred_flush "
                              "(H2D over PCIe inside the timed region); exact offsets: tests/test_gpu_fullsize.py")
                line["config2_16gib_fed"] = c2
                del h2
            except Exception as e:
                line["config2_16gib_fed"] = {"error": repr(e)}
            # configs[4]: expected chunk size 2-64 KiB, bounds off / on (min D/4, max 8D), over 10
            # backup-style snapshots of a 1 GiB master as one 10 GiB stream in HBM; at D = 8 KiB
            # also chunk -> SHA-256 per chunk -> dedup index on the device, with the dedup ratio
            try:
                sys.path.insert(0, os.path.join(ROOT, "tools"))
                import snapshots as SN
                n4 = 1 << 30
                big = torch.empty(10 * n4, dtype=torch.uint8, device=dev)
                for sidx in range(10):
                    SN.build_snapshot(big[sidx * n4:(sidx + 1) * n4], 6, sidx)
                bcap = 10 * n4 // 1024 + 65536
                bo = torch.empty(bcap, dtype=torch.int64, device=dev)
                bn = torch.zeros(1, dtype=torch.int64, device=dev)
                pts = []
                for D in (2048, 4096, 8192, 16384, 32768, 65536):
                    for bnd in (False, True):
                        cx = pkg.Chunker(pkg.Params(divisor=D, min_size=D // 4 if bnd else 0,
                                                    max_size=8 * D if bnd else 0), device=local)
                        cx.chunk_async(big, bo, bn)
                        torch.cuda.synchronize()
                        q0.record(stream)
                        cx.chunk_async(big, bo, bn)
                        q1.record(stream)
                        torch.cuda.synchronize()
                        pts.append({"D": D, "bounds": [D // 4, 8 * D] if bnd else "off",
                                    "gbs": round(10 * n4 / (q0.elapsed_time(q1) * 1e-3) / 1e9, 1),
                                    "mean_chunk": round(10 * n4 / (int(bn.item()) + 1))})
                        if D == 8192 and not bnd:
                            bd = torch.empty((bcap + 1) * 32, dtype=torch.uint8, device=dev)
                            for it in range(2):
                                cx.index_reset(10 * n4 // 4096)
                                torch.cuda.synchronize()
                                q0.record(stream)
                                cx.chunk_async(big, bo, bn)
                                cx.hash_chunks_async(big, bo, bn, bd)
                                cx.index_insert_async(bd, bo, bn, 10 * n4)
                                q1.record(stream)
                                torch.cuda.synchronize()
                            stx = cx.index_stats()
                            pipe = {"gbs": round(10 * n4 / (q0.elapsed_time(q1) * 1e-3) / 1e9, 1),
                                    "dedup_ratio": round(10 * n4 / max(1, stx["new_bytes"]), 3),
                                    "generator_expectation": round(10 / (1 + sum(synthgen.SNAPSHOT_P[1:])), 3)}
                            del bd
                        del cx
                line["config4_sweep"] = {"points": pts, "pipeline_8k": pipe, "unit": "GB/s",
                                         "note": "configs[4]: 10 snapshots x 1 GiB (1 MiB segments replaced with "
                                                 "p = 5-25 %) chunked as one 10 GiB stream per point; pipeline_8k = "
                                                 "chunk -> SHA-256 -> dedup index at D = 8 KiB, bounds off"}
                del big, bo
                torch.cuda.empty_cache()
            except Exception as e:
                line["config4_sweep"] = {"error": repr(e)}
        except Exception as e:  # side numbers must never break the headline line
            line["extra_error"] = repr(e)

    # ---- CPU baselines on this box's host cores (rank 0, N = 1 only; measured above in a fresh
    # process before the CUDA work): the oracle, and the paper's §5.1 multithreaded chunker
    if cpu is not None:
        line["cpu_baseline"] = cpu.get("cpu_baseline")
        if "cpu_chunker" in cpu:
            cc = dict(cpu["cpu_chunker"])
            if "count" in cc:
                cc["matches_gpu_count"] = cc.pop("count") == n_cand
            line["cpu_chunker"] = cc

    if rank == 0:
        print(json.dumps(line), flush=True)
    if world > 1:
        dist.barrier()
        dist.destroy_process_group()


if __name__ == "__main__":
    main()

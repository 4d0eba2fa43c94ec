// size_bound.cuh — the min/max chunk-size rule on the device.
//
// The rule (readings Q12-Q15), over ascending candidates c with state
// s = the last cut (0 at the stream start):
//     while c - s > max: s += max, emit s          (forced cut: no acceptable marker in max bytes)
//     if c - s >= min:   emit c, s = c             (markers closer than min are dropped)
//   and at the end of the stream N: while N - s > max: s += max, emit s (s < N).
// It is sequential in s, but the state is a single number and two runs over the same
// candidates that ever reach the same s stay identical afterwards.  The parallel form
// (exact for any input):
//   sb_spec_check  block b of SB_B candidates runs speculatively from g_b = c[first-1] (i.e.
//             "the previous candidate was accepted"; block 0 from the true initial state)
//             -> spec exit state, spec count; and, in lockstep, from e_b = the spec exit of
//             block b-1 (recomputed by the same thread) until the two states coincide (sync)
//             -> count delta; no sync -> not ok.
//             Each CTA also reduces its blocks' counts and sync flags (cta_sum, cta_ok).
//   sb_plan   one CTA: if every block synced, entries = spec exits and the offsets are a scan
//             of the per-CTA sums (two-level scan: sb_emit adds the in-CTA prefix); otherwise
//             warp 0 walks the blocks in order, re-walking the ones whose assumed entry does not
//             hold (exact; serial only through those blocks) and writes every entry and offset.
//   sb_emit   every block re-runs from its true entry and writes its cuts at its offset; one
//             extra thread writes the forced cuts after the last candidate.
// Streaming: `fin` = 1 for a whole stream (cuts < end = N); fin = 0 for a fed piece: an accepted
// candidate exactly at `end` is held (emitted first by the next piece or dropped by the flush),
// forced cuts strictly before `end` are emitted.
#pragma once
#include "kernels.cuh"

namespace shred {

// Block size B (candidates per speculative block, one thread each).  A block syncs at its first
// candidate c >= g + min (g = its guessed entry; accepted from the true entry s <= g too), so it
// fails only if all B candidates lie within min of g (~P(Poisson(min/D) >= B) on random data); the
// repair passes then fix the chain.  B = 8 (twice the threads, half the chain) is faster when
// min <= D/2 (1 GiB at the LBFS bounds 561 -> 552 us, 256 MiB 175 -> 164 us); at min >= D its
// repairs need more passes (min = D 0.78 -> 0.93 ms), so B = 16 there (launch_size_bound picks).
// A/B log: profiles/r02_ab_small_bounded.txt.
#ifndef SHRED_SB_B
#define SHRED_SB_B 16
#endif
constexpr int SB_B = SHRED_SB_B;      // the large-min / one-CTA block size
constexpr int SB_B_SMALL = 8;         // min <= D/2
constexpr int SB_THREADS = 128;

struct SBArgs {
    const uint64_t *cand;           // ascending candidates
    const uint64_t *n_dev;          // candidate count (device), or null -> n_host
    uint64_t n_host;
    uint64_t n_cap;                 // a device count is clamped to this (the list's capacity)
    uint64_t minsz, maxsz;          // maxsz 0 = inf
    uint64_t end;                   // stream end (fin = 1) or current fed end (fin = 0)
    int fin;
    uint64_t *spec_exit, *spec_cnt, *entry, *offs;   // [nb] each
    int64_t *delta;
    uint32_t *ok;
    uint64_t *cta_sum, *cta_ok, *cta_off;            // [ncta] per spec_check CTA (two-level scan)
    uint64_t *dst; uint64_t dst_cap;
    Aux *aux;                       // s, held, held_val, out_pos (streaming state)
    uint32_t tile;                  // blocks per tile = the threads of the CTA running the phases
    uint64_t *n_out;                // one-shot chain: the caller's count, written with the final state
};
// The call end of a one-shot chain (k_call_end's job) where the final state is written.
__device__ __forceinline__ void sb_call_end(const SBArgs &A) {
    if (A.n_out) {
        *A.n_out = A.aux->out_pos;
        if (A.aux->out_pos > A.dst_cap) A.aux->overflow = 1;
    }
}

__device__ __forceinline__ uint64_t sb_n(const SBArgs &A) {
    if (!A.n_dev) return A.n_host;
    const uint64_t n = *A.n_dev;
    return n < A.n_cap ? n : A.n_cap;
}

// One candidate: returns the number of cuts emitted (forced + accepted, held excluded).
template <class Emit>
__device__ __forceinline__ uint64_t sb_step(uint64_t &s, uint64_t c, const SBArgs &A, int &held, Emit emit) {
    uint64_t k = 0;
    if (A.maxsz && c - s > A.maxsz) {
        const uint64_t m = (c - s - 1) / A.maxsz;     // forced cuts s+max, ..., s+m*max (all < c)
        for (uint64_t j = 1; j <= m; ++j) emit(s + j * A.maxsz);
        s += m * A.maxsz;
        k += m;
    }
    if (c - s >= A.minsz) {
        s = c;
        if (!A.fin && c == A.end) held = 1;
        else { emit(c); ++k; }
    }
    return k;
}
struct NoEmit { __device__ void operator()(uint64_t) const {} };

// Forced cuts after the last candidate, strictly before `end`.
__device__ __forceinline__ uint64_t sb_tail_count(uint64_t s, const SBArgs &A) {
    if (!A.maxsz || A.end <= s) return 0;
    return (A.end - s - 1) / A.maxsz;
}

// sb_spec + sb_check fused: thread b runs the speculation of block b-1 (to get its exit X),
// then block b from its own guess and, in lockstep, from X until the two states coincide.
// Tiles of SB_THREADS blocks; CTA i takes tiles i, i + gridDim.x, ... (the grid is sized for the
// capacity bound, the tile count comes from the true count on the device).
// The phases are device functions so that one CTA can run them back to back (sb_one): tiles of
// A.tile = blockDim.x blocks, CTA `bid` of `nblk` takes tiles bid, bid + nblk, ...
template <int B>
__device__ __forceinline__ void sb_spec_body(const SBArgs &A, uint32_t bid, uint32_t nblk) {
    const uint64_t n = sb_n(A);
    const uint64_t nb = (n + B - 1) / B;
    const uint32_t T = blockDim.x;
    for (uint64_t tile = bid; tile * T < nb; tile += nblk) {
    const uint64_t b = tile * T + threadIdx.x;
    uint64_t cnt = 0;
    bool synced = true;
    if (b < nb) {
        const uint64_t first = b * B, last = min(n, first + B);
        uint64_t v[B], w[B];
        uint64_t X = 0;
        int hX = 0;
        // both blocks' candidates in one round trip (the previous block's for its speculation)
#pragma unroll
        for (int j = 0; j < B; ++j) v[j] = (first + j < last) ? A.cand[first + j] : 0ull;
        const uint64_t pf = b ? first - B : 0;
#pragma unroll
        for (int j = 0; j < B; ++j) w[j] = b ? A.cand[pf + j] : 0ull;
        const uint64_t s0 = A.aux->s;
        X = (b > 1) ? A.cand[pf - 1] : s0;
        if (b) {                              // speculation of block b-1 (its guess, or exact for 0)
#pragma unroll
            for (int j = 0; j < B; ++j) sb_step(X, w[j], A, hX, NoEmit{});
        }
        uint64_t sg = b ? w[B - 1] : s0;   // this block's guess: the previous candidate accepted
        int hg = 0, ht = 0;
        uint64_t cg = 0;
        int64_t ct = 0, cg_sync = 0;
        synced = (b == 0) || (X == sg && hX == 0);
        uint64_t st = X;
#pragma unroll
        for (int j = 0; j < B; ++j) {
            if (first + j < last) {
                const uint64_t k = sb_step(sg, v[j], A, hg, NoEmit{});
                cg += k;
                if (!synced) {
                    ct += (int64_t)sb_step(st, v[j], A, ht, NoEmit{});
                    cg_sync += (int64_t)k;
                    synced = (st == sg) && (ht == hg);
                }
            }
        }
        A.spec_exit[b] = sg;
        A.spec_cnt[b] = cg;
        A.ok[b] = synced ? 1u : 0u;
        A.delta[b] = ct - cg_sync;
        cnt = (uint64_t)((int64_t)cg + ct - cg_sync);
    }
    // per-CTA sum of the counts (valid if every block synced) and AND of the sync flags
    __shared__ uint64_t red[32];
    uint64_t x = cnt;
    for (int d = 16; d; d >>= 1) x += __shfl_xor_sync(0xffffffffu, x, d);
    const int all = __syncthreads_and(synced ? 1 : 0);
    if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = x;
    __syncthreads();
    if (threadIdx.x == 0) {
        uint64_t t = 0;
        for (uint32_t w = 0; w < T / 32; ++w) t += red[w];
        A.cta_sum[tile] = t;
        A.cta_ok[tile] = all ? 1u : 0u;
    }
    __syncthreads();                          // red reused by the next tile
    }
}
template <int B>
__global__ void __launch_bounds__(SB_THREADS) sb_spec_check(SBArgs A) {
    pdl_entry();
    if (A.aux->dense) return;                 // the candidates did not fit: sb_dense runs
    sb_spec_body<B>(A, blockIdx.x, gridDim.x);
}

// One CTA: entries, offsets, totals and the streaming state.  Each thread owns a contiguous
// range of blocks; one block scan of the range sums gives every block's offset.
template <int B>
__device__ __forceinline__ void sb_plan_body(const SBArgs &A) {
    __shared__ uint64_t wsum[33];
    const uint64_t n = sb_n(A);
    const uint32_t nb = (uint32_t)((n + B - 1) / B);
    const uint32_t tid = threadIdx.x;
    const uint32_t nc = (nb + A.tile - 1) / A.tile;                 // tiles with blocks
    const uint32_t per = (nc + blockDim.x - 1) / blockDim.x;
    const uint32_t ca = min(nc, tid * per), cb = min(nc, ca + per);
    uint64_t sum = 0;
    uint32_t bad = 0;
    for (uint32_t c = ca; c < cb; ++c) {
        sum += A.cta_sum[c];
        bad |= (uint32_t)(A.cta_ok[c] ^ 1u);
    }
    const int all_ok = __syncthreads_and(bad == 0);
    Aux *aux = A.aux;
    const uint64_t held_prev = aux->held;
    const uint64_t base0 = aux->out_pos + held_prev;
    if (all_ok) {
        uint64_t incl = sum;
        for (int d = 1; d < 32; d <<= 1) {
            uint64_t u = __shfl_up_sync(0xffffffffu, incl, d);
            if ((tid & 31) >= (uint32_t)d) incl += u;
        }
        if ((tid & 31) == 31) wsum[tid >> 5] = incl;
        __syncthreads();
        if (tid == 0) {
            uint64_t r = 0;
            for (uint32_t w = 0; w < (blockDim.x >> 5); ++w) { uint64_t x = wsum[w]; wsum[w] = r; r += x; }
            wsum[32] = r;
        }
        __syncthreads();
        uint64_t off = base0 + wsum[tid >> 5] + incl - sum;
        for (uint32_t c = ca; c < cb; ++c) {        // sb_emit adds the in-CTA prefix
            A.cta_off[c] = off;
            off += A.cta_sum[c];
        }
        const uint64_t carry = wsum[32];
        if (tid == 0) {
            const uint64_t s_last = nb ? A.spec_exit[nb - 1] : aux->s;
            // the held flag of the piece: the last candidate accepted exactly at `end`
            int held_new = 0;
            if (!A.fin && n > 0 && A.cand[n - 1] == A.end && s_last == A.end) held_new = 1;
            const uint64_t mt = sb_tail_count(s_last, A);
            if (held_prev && aux->out_pos < A.dst_cap) A.dst[aux->out_pos] = aux->held_val;
            A.entry[0] = aux->s;                  // block 0's entry (the others: spec exits)
            aux->out_pos = base0 + carry + mt;
            aux->s = s_last + mt * A.maxsz;
            aux->held = (uint64_t)held_new;
            aux->held_val = held_new ? A.end : 0;
            aux->total = carry + mt;
            aux->sb_fast = 1;
            sb_call_end(A);
            A.offs[nb] = base0 + carry;           // the tail's forced cuts start here
            A.entry[nb] = s_last;
        }
        return;
    }
    // ---- parallel repair (some block did not sync with its speculation): Jacobi passes over
    // super-blocks of G blocks, each re-run from the exit of the previous one as currently known
    // (only when that entry changed), until no exit changes -- exact at the fixed point, where
    // every super-block ran from its true entry.  A block whose speculation failed usually
    // changes only the next block or two (min ~ D: converged at G = 1 in 2-3 passes).  Long
    // chains of unsynced blocks (min >> D: a cut needs a gap >= min from the leading state) need
    // super-blocks long enough to re-sync: G = 32 (min = 8D); beyond that the serial walk below.
#ifndef SHRED_SB_REPAIR_LEVELS
#define SHRED_SB_REPAIR_LEVELS 2      // G = 1, 32 (A/B: 0 = straight to the serial walk; 3 adds G = 1024,
                                      // which cost more than the walk when it fails: min = 16D 4.1 -> 8.0 ms)
#endif
    for (int lvl = 0; lvl < SHRED_SB_REPAIR_LEVELS; ++lvl) {
        const uint32_t G = lvl == 0 ? 1u : lvl == 1 ? 32u : 1024u;     // blocks per super-block
        const uint32_t ns = (nb + G - 1) / G;                  // super-blocks
        if (lvl > 0 && ns < 4) break;                           // no parallelism left: walk
        uint64_t *Ea = A.entry, *Eb = A.cta_sum, *Cn = A.cta_ok, *Used = A.offs;   // scratch
        const uint32_t T = blockDim.x, ps = (ns + T - 1) / T;
        SHRED_ASSERT(ns <= nb + 1 && nb + 1 <= A.n_cap / B + 2);
        const uint32_t sa = min(ns, tid * ps), se = min(ns, sa + ps);
        for (uint32_t k = sa; k < se; ++k) { Ea[k] = A.spec_exit[min(nb, (k + 1) * G) - 1]; Used[k] = ~0ull; }
        __syncthreads();
        const int passes = lvl == 0 ? 12 : lvl == 1 ? 6 : 3;   // a pass at G = 1024 costs ~0.35 ms
        int conv = 0, p = 0;
        for (; p < passes && !conv; ++p) {
            const uint64_t *src = (p & 1) ? Eb : Ea;
            uint64_t *dst = (p & 1) ? Ea : Eb;
            int changed = 0;
            for (uint32_t k = sa; k < se; ++k) {
                const uint64_t e = k ? src[k - 1] : aux->s;
                if (e != Used[k]) {
                    const uint64_t first = (uint64_t)k * G * B, last = min(n, first + (uint64_t)G * B);
                    uint64_t x = e;
                    int h = 0;
#pragma unroll 4
                    for (uint64_t j = first; j < last; ++j) sb_step(x, A.cand[j], A, h, NoEmit{});
                    Used[k] = e;
                    changed |= (x != src[k]) ? 1 : 0;
                    dst[k] = x;
                } else {
                    dst[k] = src[k];
                }
            }
            conv = !__syncthreads_or(changed);
        }
        if (!conv) { __syncthreads(); continue; }
        const uint64_t *E = (p & 1) ? Eb : Ea;                  // the last pass's output
        const uint64_t s_last = ns ? E[ns - 1] : aux->s;
        __syncthreads();                                        // E (= entry) is rewritten below
        // every super-block from its true entry once more: per-block entries and counts
        for (uint32_t k = sa; k < se; ++k) {
            uint64_t x = Used[k];
            int h = 0;
            for (uint32_t b = k * G; b < min(nb, (k + 1) * G); ++b) {
                const uint64_t first = (uint64_t)b * B, last = min(n, first + B);
                A.entry[b] = x;
                uint64_t cnt = 0;
                for (uint64_t j = first; j < last; ++j) cnt += sb_step(x, A.cand[j], A, h, NoEmit{});
                Cn[b] = cnt;
            }
        }
        __syncthreads();
        // offsets: exclusive scan of the block counts (contiguous ranges per thread)
        const uint32_t pb = (nb + T - 1) / T, ba = min(nb, tid * pb), bb = min(nb, ba + pb);
        uint64_t rs = 0;
        for (uint32_t b = ba; b < bb; ++b) rs += Cn[b];
        uint64_t incl = rs;
        for (int d = 1; d < 32; d <<= 1) {
            const uint64_t u = __shfl_up_sync(0xffffffffu, incl, d);
            if ((tid & 31) >= (uint32_t)d) incl += u;
        }
        if ((tid & 31) == 31) wsum[tid >> 5] = incl;
        __syncthreads();
        if (tid == 0) {
            uint64_t r = 0;
            for (uint32_t w = 0; w < (T >> 5); ++w) { const uint64_t x = wsum[w]; wsum[w] = r; r += x; }
            wsum[32] = r;
        }
        __syncthreads();
        uint64_t o = base0 + wsum[tid >> 5] + incl - rs;
        for (uint32_t b = ba; b < bb; ++b) { A.offs[b] = o; o += Cn[b]; }
        if (tid == 0) {
            const uint64_t carry = wsum[32];
            const int held_new = (!A.fin && n > 0 && A.cand[n - 1] == A.end && s_last == A.end) ? 1 : 0;
            const uint64_t mt = sb_tail_count(s_last, A);
            aux->sb_fast = 0;
            if (held_prev && aux->out_pos < A.dst_cap) A.dst[aux->out_pos] = aux->held_val;
            A.offs[nb] = base0 + carry;
            A.entry[nb] = s_last;
            aux->total = carry + mt;
            aux->out_pos = base0 + carry + mt;
            aux->s = s_last + mt * A.maxsz;
            aux->held = (uint64_t)held_new;
            aux->held_val = held_new ? A.end : 0;
            sb_call_end(A);
        }
        return;
    }
    // ---- sequential fallback (no parallel form converged): exact.  Warp 0 runs the rule over
    // every candidate in order, 32 at a time by ballot: the first candidate (in order) that
    // forces a cut or is accepted from the current state is the next one that changes it, and
    // every candidate before it drops out with no effect -- one ballot per block of B
    // candidates plus one step per cut.  Block entries and offsets are recorded at the block boundaries.  The other
    // warps stage the next window of candidates in shared memory (double-buffered).
    static_assert(32 % B == 0, "the ballot walk records a block boundary every B candidates");
    constexpr uint32_t SBW = 2048;                          // candidates per window
    __shared__ uint64_t wc[2][SBW];
    const uint32_t nwin = (uint32_t)((n + SBW - 1) / SBW);
    auto stage = [&](uint32_t wi, int buf, uint32_t t, uint32_t nt) {
        const uint64_t c0 = (uint64_t)wi * SBW;
        for (uint32_t i = t; i < SBW; i += nt)
            if (c0 + i < n) wc[buf][i] = A.cand[c0 + i];
    };
    if (nwin) stage(0, 0, tid, blockDim.x);
    __syncthreads();
    const uint32_t lane = tid & 31;
    uint64_t s = aux->s, off = base0;
    int held = 0;
    for (uint32_t wi = 0; wi < nwin; ++wi) {
        const int cur = (int)(wi & 1u);
        if (tid >= 32) {
            if (wi + 1 < nwin) stage(wi + 1, cur ^ 1, tid - 32, blockDim.x - 32);
        } else {
            const uint64_t c0 = (uint64_t)wi * SBW;
            const uint32_t m = (uint32_t)min((uint64_t)SBW, n - c0);
            for (uint32_t w0 = 0; w0 < m; w0 += 32) {
                const uint64_t mine = w0 + lane < m ? wc[cur][w0 + lane] : 0ull;
#pragma unroll
                for (uint32_t part = 0; part < 32u / B; ++part) {
                    const uint32_t lo = B * part, hi = min(lo + (uint32_t)B, m - w0);
                    if (lo >= hi) break;
                    const uint64_t b = (c0 + w0 + lo) / B;
                    SHRED_ASSERT(b < nb && w0 + 32 <= SBW + 32);
                    if (lane == 0) { A.entry[b] = s; A.offs[b] = off; }
                    uint32_t from = lo;
                    for (;;) {
                        const bool ev = lane >= from && lane < hi &&
                                        ((A.maxsz && mine - s > A.maxsz) || mine - s >= A.minsz);
                        const uint32_t bal = __ballot_sync(0xffffffffu, ev);
                        if (!bal) break;
                        const int jj = __ffs(bal) - 1;
                        off += sb_step(s, __shfl_sync(0xffffffffu, mine, jj), A, held, NoEmit{});
                        from = (uint32_t)jj + 1;
                    }
                }
            }
        }
        __syncthreads();
    }
    if (tid != 0) return;
    aux->sb_fast = 0;
    const uint64_t mt = sb_tail_count(s, A);
    if (held_prev && aux->out_pos < A.dst_cap) A.dst[aux->out_pos] = aux->held_val;
    A.offs[nb] = off;
    A.entry[nb] = s;
    aux->total = off - base0 + mt;
    aux->out_pos = off + mt;
    aux->s = s + mt * A.maxsz;
    aux->held = (uint64_t)held;
    aux->held_val = held ? A.end : 0;
    sb_call_end(A);
}
template <int B>
__global__ void __launch_bounds__(1024) sb_plan(SBArgs A) {
    pdl_entry();
    if (A.aux->dense) return;
    sb_plan_body<B>(A);
}

// Every block writes its cuts; thread nb writes the forced cuts after the last candidate.
template <int B>
__device__ __forceinline__ void sb_emit_body(const SBArgs &A, uint32_t bid, uint32_t nblk) {
    const uint64_t n = sb_n(A);
    const uint64_t nb = (n + B - 1) / B;
    const bool fast = A.aux->sb_fast != 0;
    const uint32_t T = blockDim.x;
    __shared__ uint64_t ws[33];
    for (uint64_t tile = bid; tile * T <= nb; tile += nblk) {
        const uint64_t b = tile * T + threadIdx.x;
        uint64_t s = 0, o = 0;
        // the block's candidates first: their round trip overlaps the offset scan below
        const uint64_t first = b * B, last = b < nb ? min(n, first + B) : first;
        uint64_t v[B];
#pragma unroll
        for (int j = 0; j < B; ++j) v[j] = (first + j < last) ? A.cand[first + j] : 0ull;
        if (fast) {
            // entry = the previous block's spec exit; offset = tile offset + in-tile exclusive prefix
            const uint64_t v = b < nb ? (uint64_t)((int64_t)A.spec_cnt[b] + A.delta[b]) : 0ull;
            uint64_t incl = v;
            for (int d = 1; d < 32; d <<= 1) {
                uint64_t u = __shfl_up_sync(0xffffffffu, incl, d);
                if ((threadIdx.x & 31) >= (uint32_t)d) incl += u;
            }
            if ((threadIdx.x & 31) == 31) ws[threadIdx.x >> 5] = incl;
            __syncthreads();
            uint64_t pre = 0;
            for (uint32_t w = 0; w < (threadIdx.x >> 5); ++w) pre += ws[w];
            __syncthreads();                  // ws reused by the next tile
            if (b == nb) { s = A.entry[nb]; o = A.offs[nb]; }
            else if (b < nb) { s = b ? A.spec_exit[b - 1] : A.entry[0]; o = A.cta_off[tile] + pre + incl - v; }
        } else if (b <= nb) {
            s = A.entry[b];
            o = A.offs[b];
        }
        if (b > nb) continue;
        uint64_t *dst = A.dst;
        const uint64_t cap = A.dst_cap;
        auto emit = [&](uint64_t v) { if (o < cap) dst[o] = v; ++o; };
        if (b == nb) {
            const uint64_t mt = sb_tail_count(s, A);
            for (uint64_t j = 1; j <= mt; ++j) emit(s + j * A.maxsz);
            continue;
        }
        int held = 0;
#pragma unroll
        for (int j = 0; j < B; ++j)
            if (first + j < last) sb_step(s, v[j], A, held, emit);
    }
}
template <int B>
__global__ void __launch_bounds__(SB_THREADS) sb_emit(SBArgs A) {
    pdl_entry();
    if (A.aux->dense) return;                 // the candidates did not fit: sb_dense runs
    sb_emit_body<B>(A, blockIdx.x, gridDim.x);
}

// ------------------------------------------------------------------------------ sb_dense
// Exact fallback when the ordered candidate list could not hold every candidate (only possible
// when some slot's list overflowed, i.e. dense candidates such as a repeated `04 D5`): one CTA
// walks the slots in stream order.  Warp 0 owns the rule state; slots whose list is complete
// are read from it, overflowed slots are re-rolled by all threads into a shared bitmap (in
// windows of SBD_WIN window ends) that warp 0 then scans in order.
constexpr int SBD_THREADS = 256;
constexpr uint64_t SBD_WIN = 1ull << 20;              // window ends per bitmap pass (128 KiB)
__device__ __forceinline__ void sb_dense_body(const Job &J, const DevParams &P, const GenTables *__restrict__ gt,
                                              uint32_t nslots, const SBArgs &A) {
    Aux *aux = A.aux;
    extern __shared__ uint32_t bm[];
    __shared__ uint64_t sT[256], sU[256];
    for (int i = threadIdx.x; i < 256; i += blockDim.x) { sT[i] = gt->T[i]; sU[i] = gt->U[i]; }
    __syncthreads();
    const int tid = threadIdx.x, lane = tid & 31;
    const bool w0 = tid < 32;
    uint64_t s = aux->s, off = aux->out_pos;
    int held = 0;
    uint64_t *dst = A.dst;
    const uint64_t cap = A.dst_cap;
    auto emit = [&](uint64_t v) { if (lane == 0 && off < cap) dst[off] = v; ++off; };
    if (aux->held) emit(aux->held_val);
    SmemGenTab tab{sT, sU};
    for (uint32_t slot = 0; slot < nslots; ++slot) {
        uint64_t a, b;
        slot_range(J.map, slot, a, b);
        const uint32_t cnt = J.counts[slot];
        if (cnt <= J.cap) {
            if (w0) {
                const uint64_t *lst = J.scratch + (uint64_t)slot * J.cap;
                for (uint32_t j = 0; j < cnt; j += 32) {
                    const uint64_t v = (j + lane < cnt) ? lst[j + lane] : 0ull;
                    const uint32_t m = min(32u, cnt - j);
                    for (uint32_t k = 0; k < m; ++k) sb_step(s, __shfl_sync(0xffffffffu, v, k), A, held, emit);
                }
            }
            continue;
        }
        for (uint64_t wa = a; wa < b; wa += SBD_WIN) {
            const uint64_t wb = min(b, wa + SBD_WIN);
            const uint32_t nw = (uint32_t)((wb - wa + 31) / 32);
            for (uint32_t i = tid; i < nw; i += blockDim.x) bm[i] = 0;
            __syncthreads();
            const uint64_t per = (wb - wa + blockDim.x - 1) / blockDim.x;
            const uint64_t ta = wa + per * tid, tb = min(wb, ta + per);
            if (ta < tb)
                roll_generic(J, P, tab, ta, tb, [&](uint64_t c) {
                    const uint64_t k = c - 1 - wa;                 // window end offset in the window
                    atomicOr(&bm[k >> 5], 1u << (k & 31));
                });
            __syncthreads();
            if (w0) {
                for (uint32_t i = 0; i < nw; ++i) {
                    uint32_t word = bm[i];
                    while (word) {
                        const int bit = __ffs(word) - 1;
                        word &= word - 1;
                        sb_step(s, wa + 32ull * i + (uint64_t)bit + 1, A, held, emit);
                    }
                }
            }
            __syncthreads();
        }
    }
    if (tid == 0) {
        const uint64_t mt = sb_tail_count(s, A);
        for (uint64_t j = 1; j <= mt; ++j) { if (off < cap) dst[off] = s + j * A.maxsz; ++off; }
        aux->total = off - aux->out_pos - aux->held;
        aux->out_pos = off;
        aux->s = s + mt * A.maxsz;
        aux->held = (uint64_t)held;
        aux->held_val = held ? A.end : 0;
        sb_call_end(A);
    }
}
__global__ void __launch_bounds__(SBD_THREADS)
sb_dense(Job J, DevParams P, const GenTables *__restrict__ gt, uint32_t nslots, SBArgs A) {
    pdl_entry();
    if (!A.aux->dense) return;
    sb_dense_body(J, P, gt, nslots, A);
}

// ------------------------------------------------------------------------------ sb_one
// A whole one-shot bounded call's size rule in ONE CTA, plus the call's state set-up and end
// (k_stream_reset / k_call_end): the chain after k_scatter is one launch instead of five.  Used
// for inputs up to SB_ONE_MAX_LEN, where the multi-CTA chain is bound by its dependent global
// round trips and launches (1 MiB: 26.5 us per call in a CUDA graph, 7.3 unbounded).
// Fast form (n <= 8,176 candidates): the candidates are loaded into shared memory once and
// the three phases of the parallel rule run there, one block of SB_B candidates per thread:
//   spec  thread b runs block b from its guess g_b = c[16b - 1] (block 0: s = 0) -> exit E_b,
//         count C_b; and, in lockstep, from X = E_{b-1} (block b-1 rerun from ITS guess by the
//         same thread) until the two states coincide -> delta_b, synced_b;
//   plan  every block synced: the true entry of block b is E_{b-1} (induction from block 0,
//         which is exact), offsets = exclusive scan of C_b + delta_b; otherwise thread 0 walks
//         the blocks in order, re-walking candidate by candidate those whose entry is not the
//         one their sync assumed;
//   emit  block b reruns from its true entry and writes its cuts; the last thread writes the
//         forced cuts after the last candidate.
// Larger counts run the global-memory phases above (sb_*_body); dense lists sb_dense_body.
constexpr int SBO_THREADS = 1024;
constexpr int SBO_B = 8;      // candidates per block in sb_one_smem (its serial walk is over <= 1,024 blocks in smem)
constexpr uint32_t SBO_SMEM_N = SBO_THREADS * SBO_B;      // 8192 candidates, 64 KiB
constexpr size_t SBO_SMEM = (size_t)SBO_SMEM_N * 8 + (size_t)SBO_THREADS * 8 * 4;
#ifndef SHRED_SB_ONE_MAX
#define SHRED_SB_ONE_MAX (256ull << 20)  // A/B: 0 = always the multi-CTA chain
#endif
constexpr uint64_t SB_ONE_MAX_LEN = SHRED_SB_ONE_MAX;
#ifndef SHRED_SB_ONE_EXPECT
#define SHRED_SB_ONE_EXPECT 8192   // 64 MiB at D = 8 KiB (A/B: sb_one 56.6 vs chain 68.8 us; 256 MiB: 253 vs 181)
#endif
constexpr uint64_t SB_ONE_EXPECT = SHRED_SB_ONE_EXPECT;  // expected candidates (len (r+1 | 1) / D) up to which sb_one runs

__device__ __forceinline__ void sb_one_smem(const SBArgs &A, uint32_t n, uint64_t *n_out, uint64_t cap,
                                            bool loaded = false) {
    extern __shared__ uint64_t sm64[];
    uint64_t *sc = sm64;                                   // candidates [n]
    uint64_t *ex = sc + SBO_SMEM_N;                        // spec exit E_b
    uint64_t *cn = ex + SBO_THREADS;                       // count along the true path (synced)
    uint64_t *en = cn + SBO_THREADS;                       // true entry
    uint64_t *of = en + SBO_THREADS;                       // output offset
    __shared__ uint32_t okb[SBO_THREADS];
    __shared__ uint64_t wsum[SBO_THREADS / 32 + 1];
    const uint32_t tid = threadIdx.x;
    SHRED_ASSERT(n <= SBO_SMEM_N - SBO_B && blockDim.x == SBO_THREADS);
    if (!loaded)
        for (uint32_t i = tid; i < n; i += SBO_THREADS) sc[i] = A.cand[i];
    __syncthreads();
    const uint32_t nb = (n + SBO_B - 1) / SBO_B;
    const uint32_t b = tid;
    int h0 = 0;
    uint64_t cnt = 0;
    bool synced = true;
    if (b < nb) {
        const uint32_t first = b * SBO_B, last = min(n, first + SBO_B);
        uint64_t X = 0;
        if (b) {
            const uint32_t pf = first - SBO_B;
            X = (b - 1) ? sc[pf - 1] : 0ull;
            for (uint32_t j = pf; j < first; ++j) sb_step(X, sc[j], A, h0, NoEmit{});
        }
        uint64_t sg = b ? sc[first - 1] : 0ull, st = X;
        uint64_t cg = 0;
        int64_t ct = 0, cgs = 0;
        synced = (b == 0) || (X == sg);
        for (uint32_t j = first; j < last; ++j) {
            const uint64_t k = sb_step(sg, sc[j], A, h0, NoEmit{});
            cg += k;
            if (!synced) {
                ct += (int64_t)sb_step(st, sc[j], A, h0, NoEmit{});
                cgs += (int64_t)k;
                synced = st == sg;
            }
        }
        ex[b] = sg;
        cnt = (uint64_t)((int64_t)cg + ct - cgs);
        cn[b] = cnt;
        okb[b] = synced ? 1u : 0u;
    }
    const int all_ok = __syncthreads_and(synced ? 1 : 0);
    if (all_ok) {
        uint64_t incl = cnt;                               // block exclusive scan of the counts
        for (int d = 1; d < 32; d <<= 1) {
            const uint64_t u = __shfl_up_sync(0xffffffffu, incl, d);
            if ((tid & 31) >= (uint32_t)d) incl += u;
        }
        if ((tid & 31) == 31) wsum[tid >> 5] = incl;
        __syncthreads();
        if (tid == 0) {
            uint64_t r = 0;
            for (int w = 0; w < SBO_THREADS / 32; ++w) { const uint64_t x = wsum[w]; wsum[w] = r; r += x; }
            wsum[SBO_THREADS / 32] = r;
        }
        __syncthreads();
        if (b < nb) { of[b] = wsum[tid >> 5] + incl - cnt; en[b] = b ? ex[b - 1] : 0ull; }
        if (tid == 0) { of[nb] = wsum[SBO_THREADS / 32]; en[nb] = nb ? ex[nb - 1] : 0ull; }
    } else if (tid == 0) {
        // exact sequential walk: a block keeps its spec result if its true entry is the state
        // its sync assumed (E_{b-1}) and it synced, else it is re-walked
        uint64_t s = 0, off = 0;
        int h = 0;
        for (uint32_t k = 0; k < nb; ++k) {
            en[k] = s; of[k] = off;
            if (k == 0 || (okb[k] && s == ex[k - 1])) {
                off += cn[k];
                s = ex[k];
            } else {
                const uint32_t first = k * SBO_B, last = min(n, first + SBO_B);
                for (uint32_t j = first; j < last; ++j) off += sb_step(s, sc[j], A, h, NoEmit{});
            }
        }
        en[nb] = s; of[nb] = off;
    }
    __syncthreads();
    uint64_t *dst = A.dst;
    if (b <= nb) {
        uint64_t s = en[b], o = of[b];
        auto emit = [&](uint64_t v) { if (o < cap) dst[o] = v; ++o; };
        if (b == nb) {
            const uint64_t mt = sb_tail_count(s, A);
            for (uint64_t j = 1; j <= mt; ++j) emit(s + j * A.maxsz);
            Aux *aux = A.aux;                              // the call's end (k_call_end)
            aux->out_pos = o; aux->total = o;
            aux->s = s + mt * A.maxsz; aux->held = 0; aux->held_val = 0;
            *n_out = o;
            if (o > cap) aux->overflow = 1;
        } else {
            const uint32_t first = b * SBO_B, last = min(n, first + SBO_B);
            int h = 0;
            for (uint32_t j = first; j < last; ++j) sb_step(s, sc[j], A, h, emit);
        }
    }
}

__global__ void __launch_bounds__(SBO_THREADS)
sb_one(Job J, DevParams P, const GenTables *__restrict__ gt, uint32_t nslots, SBArgs A, uint64_t *n_out,
       uint64_t cap) {
    pdl_entry();
    Aux *aux = A.aux;
    const uint64_t dense = aux->dense, n = sb_n(A);
    if (!dense && n <= SBO_SMEM_N - SBO_B) {                // nb < SBO_THREADS: thread nb writes the tail
        sb_one_smem(A, (uint32_t)n, n_out, cap);
        return;
    }
    __syncthreads();                                       // every thread has read the state
    if (threadIdx.x == 0) { aux->s = 0; aux->held = 0; aux->held_val = 0; aux->out_pos = 0; }
    __syncthreads();
    if (dense) {
        sb_dense_body(J, P, gt, nslots, A);
    } else {
        sb_spec_body<SB_B>(A, 0, 1);
        __syncthreads();
        sb_plan_body<SB_B>(A);
        __syncthreads();
        sb_emit_body<SB_B>(A, 0, 1);
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        *n_out = aux->out_pos;
        if (aux->out_pos > cap) aux->overflow = 1;
    }
}

}  // namespace shred

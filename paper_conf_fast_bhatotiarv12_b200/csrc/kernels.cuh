// kernels.cuh — sm_100a device code of the B200 content-defined chunker.
//
// The method (§2.1, §3.1): a Rabin fingerprint of every w-byte
// window (w = 48), a cut candidate c = i+1 where (fp mod D) == r, then the min/max rule.
// The fingerprint is rolled one byte at a time (L450-L454, "shifting a byte forward"):
//
//     f_i = f_{i-1} * x^8 + B[i] - B[i-w] * x^{8w}    (mod P)
//
// realised with two 256-entry tables: T (reduces the byte shifted out of the top of the
// state) and U (removes the byte leaving the window).  See DESIGN.md "Kernels".
//
//   k1_bulk<MODE,C,WCH,MK,FN>  TMA-staged hot loop (FN: w not a multiple of 16, funnel pops).  The input is viewed as a 2-D [rows][S]
//                   tensor; each consumer thread rolls CH = 2 rows (independent chains) in one
//                   basic block; rounds of 32 B per row arrive in a 2-stage shared-memory ring
//                   (SWIZZLE_32B, conflict-free LDS.128) fed by a producer warp.  T/U live in
//                   shared memory, replicated per lane so the data-dependent lookups never
//                   bank-conflict.  The marker test sets bits of a per-16-byte hit mask
//                   (ISETP + predicated OR); rare hits are appended to the row's slot list.
//                   The last CTA of the launch is the "edge" CTA: it rolls the unaligned head
//                   and the ragged tail of the range with the generic byte loop.  Every CTA
//                   ends with a block scan of its slots' counts (local offsets + group sum).
//   k1_generic      Any valid parameters, byte at a time (the generic path).
//   k_scatter       Ordered compaction: group prefix (from the group sums) + local offset,
//                   copies the per-slot lists into the destination; slots that overflowed
//                   their list re-roll their range and write directly.
//   (size_bound.cuh) the min/max rule: speculative blocks + convergence check + emit.
#pragma once
#include <cstdint>
#include <cuda.h>
#include <cuda_runtime.h>
#include <cassert>

// Device-side bounds checks (the pool closed compute-sanitizer in round 2): a -DSHRED_DEBUG=1
// build (libshred_debug.so, tools/debug_build.py) asserts the index and address invariants of the
// round-2 code paths; the GPU test suite runs against it.  Compiled out otherwise.
#ifndef SHRED_DEBUG
#define SHRED_DEBUG 0
#endif
#if SHRED_DEBUG
#define SHRED_ASSERT(c) assert(c)
#else
#define SHRED_ASSERT(c) ((void)0)
#endif

#ifndef SHRED_PRODUCER_SLEEP_NS
#define SHRED_PRODUCER_SLEEP_NS 512
#endif
#ifndef SHRED_HITMODE
#define SHRED_HITMODE 3         // 3: ISETP + predicated OR per byte (default); 0: ISETP + SEL bitmask
                                // (A/B of these and of removed variants, incl. a per-chunk LOP3.PAND
                                // predicate with replay: profiles/r01_ab_variants.txt)
#endif

namespace shred {

// K63: u64 state, deg 41..63; K40: u64 state, deg 33..40; K32: u32 state, deg 9..32;
// K32B: u32 state, deg 8/16/24/32 (whole-byte top byte)
// K32T: u32 state, deg 9..32, P = x^k + Q with the terms of Q at least 8 apart and below k-7:
// the reduction of the top byte, t(x) Q(x), is then an integer product (no carries between the
// shifted copies of t), so T costs one IMAD instead of a shared-memory lookup.
// K63T: the same for the u64 state (deg 41..63, Q's terms below 25 so t(x) Q(x) fits the low
// word; the cancel term t << k lands in the high word): two IMADs instead of an LDS.64.
enum { MODE_K63 = 1, MODE_K32 = 2, MODE_GENERIC = 3, MODE_K32B = 4, MODE_K40 = 5, MODE_K32T = 6, MODE_K63T = 7 };

#ifndef SHRED_STAGES
#define SHRED_STAGES 2   // A/B (profiles/r01_ab_variants.txt): 2 stages 1,879 GB/s > 3: 1,861 > 4: 1,854
#endif
constexpr int STAGES      = SHRED_STAGES;      // TMA ring depth (5 does not fit beside the 64 KiB table)
constexpr int BOX_ROWS    = 256;               // rows per TMA box (hardware max 256)
constexpr int TAB_BYTES   = 65536;             // replicated T|U image (256 rows x 256 B)
constexpr int GEN_THREADS = 256;

// Launch shape of the hot kernel: CH rows (independent fingerprint chains) per consumer
// thread, NTC consumer threads (+ 1 producer warp) per CTA, one CTA per SM.  A pipeline round
// brings ROUND = 64/CH bytes of every row; 4 chunks of 16 B per row per loop iteration.
#ifndef SHRED_ROUND
#define SHRED_ROUND 0   // 0: 64/CH bytes per row per TMA round; A/B: 16 (smaller stages)
#endif
template <int CH_, int NTC_, bool DW_ = false>
struct BulkCfg {
    static constexpr int CH = CH_, NTC = NTC_;
    static constexpr bool DIRECT_WARM = DW_;              // row start state by positional tables
    static constexpr int ROWS = NTC * CH;                 // rows per bulk CTA
    static constexpr int ROUND = SHRED_ROUND ? SHRED_ROUND : 64 / CH;   // bytes per row per round
    static constexpr int RPI = 64 / ROUND;                // rounds per 64-byte loop iteration
    static constexpr int CPR = ROUND / 16;                // 16-byte chunks per row per round
    static constexpr int BOX = ROWS < BOX_ROWS ? ROWS : BOX_ROWS;   // rows per TMA box
    static constexpr int STAGE = ROWS * ROUND;            // bytes per TMA stage
    static constexpr int BAR_OFF = TAB_BYTES + STAGES * STAGE;
    static constexpr int SMEM = BAR_OFF + 2048;           // + barriers/scan scratch + 1 KiB align
    static_assert(ROWS % BOX == 0 && STAGE % 1024 == 0 && (CH == 1 || CH == 2 || CH == 4) && NTC % 32 == 0 &&
                  NTC + 32 <= 1024, "shape");
};
#ifndef SHRED_K63_CH
#define SHRED_K63_CH 2
#endif
#ifndef SHRED_K63_NT
#define SHRED_K63_NT 512
#endif
#ifndef SHRED_K32_CH
#define SHRED_K32_CH 2
#endif
#ifndef SHRED_K32_NT
#define SHRED_K32_NT 512
#endif
using CfgK63 = BulkCfg<SHRED_K63_CH, SHRED_K63_NT>;
using CfgK32 = BulkCfg<SHRED_K32_CH, SHRED_K32_NT>;
// Small inputs (< ~5 MB): 128 consumers x 2 rows per CTA (two CTAs per SM fit), so the short
// rows still spread over every SM (1 MiB: 65 CTAs instead of 17; 19.8 -> 16.7 us per call).
// Its rows are 64 B, as long as the 64-byte warm-up.  DIRECT_WARM (off) computes the row start
// state directly (w independent positional-table loads) instead of by 64 dependent steps: parity
// green but slower (1 MiB 13.1 -> 13.5 us per call; the uncoalesced gathers cost more than the
// chain, which is not the critical path of a small call).
#ifndef SHRED_DIRECT_WARM
#define SHRED_DIRECT_WARM 0   // A/B: measured slower (profiles/r01_ab_variants.txt)
#endif
#ifndef SHRED_SMALL_NT
#define SHRED_SMALL_NT 128    // 128 consumers x 2 rows; 64 (128-row CTAs, 129 CTAs for 1 MiB): slower (r01_ab_variants)
#endif
using CfgSmall = BulkCfg<2, SHRED_SMALL_NT, SHRED_DIRECT_WARM != 0>;
// Long windows (w > 64, the hot kernel's WCH = 0 instances): the bytes leaving the window come
// from a second TMA tile per stage, [16 * ceil(w/16)] bytes behind the data tile, 48 bytes per row
// and round (the round's two aligned pop chunks plus the next one for the funnel), unswizzled
// (rows 48 B apart: the 8 rows of a quarter warp hit 8 distinct bank groups).
constexpr int LW_POPW = 48;
template <class C> struct LwLayout {
    static constexpr int POP_STAGE = C::ROWS * LW_POPW;
    static constexpr int BAR_OFF = TAB_BYTES + STAGES * (C::STAGE + POP_STAGE);
    static constexpr int SMEM = BAR_OFF + 2048;
};

// Slot id -> range of window-end positions.  Slots are numbered in stream order:
// [0, n_head) generic head segments, then the bulk rows, then generic tail segments.
// Slot groups (one group sum each): bulk mode: group 0 = head slots, 1 + r/rows_cta = bulk rows,
// nc + 1 = tail slots; generic-only mode (nrows == 0): group = slot / GEN_THREADS.
struct SlotMap {
    uint64_t head_start; uint64_t head_seg; uint32_t n_head;
    uint32_t nrows;      uint64_t b0;       uint64_t S;
    uint64_t tail_start; uint64_t tail_seg; uint32_t n_tail;
    uint32_t nc;         uint32_t ngroups;  // bulk CTAs; number of groups
    uint32_t rows_cta;   uint32_t pad;      // rows per bulk CTA
    uint64_t t_end;
};

__host__ __device__ __forceinline__ uint32_t slot_group(const SlotMap &m, uint32_t slot) {
    if (m.nrows == 0) return slot / GEN_THREADS;
    if (slot < m.n_head) return 0;
    slot -= m.n_head;
    if (slot < m.nrows) return 1 + slot / m.rows_cta;
    return m.nc + 1;
}

struct DevParams {              // chunking parameters as the kernels need them
    uint64_t dmask;             // D - 1 (D a power of two)
    uint64_t magic;             // r
    uint64_t kmask;             // 2^k - 1
    uint64_t divisor;           // D
    uint32_t k;                 // deg P
    uint32_t w;                 // window bytes
    uint32_t pow2;              // D is a power of two
    uint32_t marker;            // 0: fp mod D == r; 1: fp mod D <= r
};

// The marker predicate of the generic path (L247-L251, L447-L451).  The 64-bit modulo is a
// software division: keep it behind a real branch so power-of-two divisors never pay for it.
static __device__ __noinline__ uint64_t mod_u64(uint64_t f, uint64_t d) { return f % d; }
__device__ __forceinline__ bool generic_marker(uint64_t f, const DevParams &P) {
    uint64_t v;
    if (P.pow2) v = f & P.dmask;
    else v = mod_u64(f, P.divisor);
    return P.marker ? (v <= P.magic) : (v == P.magic);
}

struct Job {
    const uint8_t *src;         // src[0] is stream position p_begin
    uint64_t p_begin;
    const uint8_t *prefix;      // virtual bytes [p_begin - prefix_len, p_begin) (the carry)
    uint32_t prefix_len;
    uint32_t cap;               // per-slot list capacity
    uint64_t min_i;             // w - 1: only full windows are tested (reading Q10)
    uint64_t c_limit;           // emit c only if c < c_limit (reading Q11)
    uint32_t *counts;           // [nslots] true candidate count per slot
    uint32_t *local_off;        // [nslots] exclusive prefix of counts within the slot's group
    uint64_t *group_sum;        // [ngroups] candidates per group
    uint64_t *scratch;          // [nslots * cap] per-slot candidate lists
    SlotMap map;
};

struct GenTables { uint64_t T[256]; uint64_t U[256]; };

// Device-resident streaming / output state (one per ctx).
struct Aux {
    uint64_t total;             // candidates of the current piece (k_scatter / k_total)
    uint64_t last_cand;         // last candidate of the current piece (k_scatter)
    uint64_t out_pos;           // cuts already written by the current API call
    uint64_t s;                 // size rule: last cut (absolute)
    uint64_t held;              // 1 if a cut at exactly the previous stream end is held
    uint64_t held_val;
    uint64_t overflow;          // sticky: an output did not fit
    uint64_t dense;             // the ordered candidate list did not fit (size-rule fallback)
    uint64_t ncand;             // candidates of the current piece (k_scatter; read by sb_*)
    uint64_t sb_fast;           // sb_plan: 1 = every block synced (two-level scan offsets)
};

// Programmatic dependent launch (shred.cu pdl_launch): wait until the previous kernel of the
// stream has completed and its writes are visible, then let the next kernel start launching.
// Both are no-ops for a kernel launched without the attribute.
__device__ __forceinline__ void pdl_entry() {
    asm volatile("griddepcontrol.wait;" ::: "memory");
    asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
}
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
__device__ __forceinline__ void pdl_trigger() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }
// k1_bulk: the ctx's constant tables (written once at shred_init) are staged and the mbarriers
// initialised before griddepcontrol.wait, so that prologue overlaps the previous kernel of the
// stream; everything that reads the input or writes the job's scratch comes after the wait.
#ifndef SHRED_PDL_EARLY
#define SHRED_PDL_EARLY 1
#endif

// ------------------------------------------------------------------------------ PTX helpers
__device__ __forceinline__ uint32_t smem_u32(const void *p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}
__device__ __forceinline__ uint2 lds64(uint32_t a) {
    uint2 v;
    asm volatile("ld.shared.v2.u32 {%0, %1}, [%2];" : "=r"(v.x), "=r"(v.y) : "r"(a));
    return v;
}
__device__ __forceinline__ uint32_t lds32(uint32_t a) {
    uint32_t v;
    asm volatile("ld.shared.u32 %0, [%1];" : "=r"(v) : "r"(a));
    return v;
}
__device__ __forceinline__ uint4 lds128(uint32_t a) {
    uint4 v;
    asm volatile("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];"
                 : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(a));
    return v;
}
__device__ __forceinline__ void mbar_init(uint32_t bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" :: "r"(bar), "r"(count) : "memory");
}
__device__ __forceinline__ void mbar_expect_tx(uint32_t bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;"
                 :: "r"(bar), "r"(bytes) : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint32_t bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" :: "r"(bar) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint32_t bar, uint32_t parity) {
    asm volatile("{\n"
                 ".reg .pred P1;\n"
                 "LAB_WAIT:\n"
                 "mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n"
                 "@P1 bra DONE;\n"
                 "bra LAB_WAIT;\n"
                 "DONE:\n"
                 "}\n" :: "r"(bar), "r"(parity) : "memory");
}
__device__ __forceinline__ bool mbar_try_wait(uint32_t bar, uint32_t parity) {
    uint32_t ok;
    asm volatile("{\n"
                 ".reg .pred P1;\n"
                 "mbarrier.try_wait.parity.shared::cta.b64 P1, [%1], %2;\n"
                 "selp.u32 %0, 1, 0, P1;\n"
                 "}\n" : "=r"(ok) : "r"(bar), "r"(parity) : "memory");
    return ok != 0;
}
// Producer-side wait: back off with nanosleep so the spinning warp does not steal issue slots
// from the consumer warps of its SM sub-partition (ncu r01: the spin was ~12% of all issued
// instructions).
__device__ __forceinline__ void mbar_wait_sleep(uint32_t bar, uint32_t parity) {
    while (!mbar_try_wait(bar, parity)) __nanosleep(SHRED_PRODUCER_SLEEP_NS);
}
// 1-D bulk copy global -> shared (TMA engine), completing on an mbarrier.
__device__ __forceinline__ void bulk_g2s(uint32_t dst, const void *src, uint32_t bytes, uint32_t bar) {
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
                 :: "r"(dst), "l"(src), "r"(bytes), "r"(bar) : "memory");
}
__device__ __forceinline__ void tma_load_2d(uint32_t dst, const CUtensorMap *map, int x, int y,
                                            uint32_t bar) {
    asm volatile("cp.async.bulk.tensor.2d.shared::cluster.global.mbarrier::complete_tx::bytes"
                 " [%0], [%1, {%2, %3}], [%4];"
                 :: "r"(dst), "l"(map), "r"(x), "r"(y), "r"(bar) : "memory");
}

// ------------------------------------------------------------------------------ generic roll
// Byte at absolute stream position `pos` of a job: src, else the carried prefix, else 0
// (before the stream start; zero bytes leave a zero state unchanged, U[0] = 0).
__device__ __forceinline__ uint32_t job_byte(const Job &J, uint64_t pos) {
    if (pos >= J.p_begin) return J.src[pos - J.p_begin];
    uint64_t lo = J.p_begin - J.prefix_len;
    if (pos >= lo) return J.prefix[pos - lo];
    return 0u;
}

// Sequential reader of a job's bytes: 16-byte aligned vector loads (generic address space: the
// source is global memory or a shared-memory staging buffer), one load per 16 positions instead
// of a byte load per position (every lane of a warp reads its own segment, so each byte load
// touched 32 lines); byte loads for the carried prefix and for the block that reaches `lim`.
struct ByteStream {
    const uint8_t *lim;                 // end of the bytes this reader may touch
    const uint8_t *blk = nullptr;       // the 16-byte block held in v
    uint4 v;
    __device__ __forceinline__ uint32_t get(const Job &J, uint64_t pos) {
        if (pos < J.p_begin) return job_byte(J, pos);
        const uint8_t *a = J.src + (pos - J.p_begin);
        const uint8_t *b = reinterpret_cast<const uint8_t *>(reinterpret_cast<uintptr_t>(a) & ~(uintptr_t)15);
        if (b + 16 > lim) return *a;
        if (b != blk) { blk = b; v = *reinterpret_cast<const uint4 *>(b); }
        const uint32_t k = (uint32_t)(reinterpret_cast<uintptr_t>(a) & 15u);
        const uint32_t w = (k & 8u) ? ((k & 4u) ? v.w : v.z) : ((k & 4u) ? v.y : v.x);
        return __byte_perm(w, 0u, 0x4440u | (k & 3u));
    }
};

// Roll the exact fingerprint over window ends [seg_start, seg_end) from a zero state
// w-1 bytes earlier (or the first available byte), calling emit(c) for every candidate.
// Plain byte-at-a-time form: f <- ((f << 8) mod x^k) ^ b ^ T[top byte] ^ U[B[pos-w]].
// VEC: bytes through ByteStream (long segments in global memory); else one load per byte (the
// edge CTA's short segments staged in shared memory, where the per-byte latency chain matters:
// 1 MiB call 14.3 -> 18.1 us with ByteStream there).
template <class Tab, class Emit, bool VEC = true>
__device__ __forceinline__ void roll_generic(const Job &J, const DevParams &P, const Tab &tab,
                                             uint64_t seg_start, uint64_t seg_end, Emit emit) {
    const uint64_t lo = J.p_begin - J.prefix_len;
    const uint64_t warm = (uint64_t)P.w - 1u;
    uint64_t p = (seg_start >= lo + warm) ? seg_start - warm : lo;
    uint64_t f = 0;
    const uint8_t *lim = seg_end > J.p_begin ? J.src + (seg_end - J.p_begin) : J.src;
    ByteStream in{lim}, out{lim};
    for (uint64_t pos = p; pos < seg_end; ++pos) {
        uint32_t b = VEC ? in.get(J, pos) : job_byte(J, pos);
        uint32_t t = (uint32_t)(f >> (P.k - 8u)) & 0xFFu;
        f = ((f << 8) & P.kmask) ^ (uint64_t)b ^ tab.T(t);
        if (pos >= p + P.w) f ^= tab.U(VEC ? out.get(J, pos - P.w) : job_byte(J, pos - P.w));
        if (pos >= seg_start && pos >= J.min_i && generic_marker(f, P) && pos + 1 < J.c_limit)
            emit(pos + 1);
    }
}

struct SmemGenTab {
    const uint64_t *t, *u;
    __device__ uint64_t T(uint32_t i) const { return t[i]; }
    __device__ uint64_t U(uint32_t i) const { return u[i]; }
};
struct GlobalGenTab {
    const GenTables *g;
    __device__ uint64_t T(uint32_t i) const { return __ldg(&g->T[i]); }
    __device__ uint64_t U(uint32_t i) const { return __ldg(&g->U[i]); }
};

__device__ __forceinline__ void slot_range(const SlotMap &m, uint32_t slot, uint64_t &a, uint64_t &b) {
    if (slot < m.n_head) {
        a = m.head_start + (uint64_t)slot * m.head_seg;
        uint64_t lim = m.nrows ? m.b0 : (m.n_tail ? m.tail_start : m.t_end);
        b = a + m.head_seg; if (b > lim) b = lim;
        return;
    }
    slot -= m.n_head;
    if (slot < m.nrows) { a = m.b0 + (uint64_t)slot * m.S; b = a + m.S; return; }
    slot -= m.nrows;
    a = m.tail_start + (uint64_t)slot * m.tail_seg;
    b = a + m.tail_seg; if (b > m.t_end) b = m.t_end;
}

// ------------------------------------------------------------------------------ block scan
// Exclusive scan of one u32 per thread over the first `nthr` threads (a multiple of 32) of the
// CTA, using named barrier `bar` and `ws` (>= 33 u32 of shared memory).  Returns the
// exclusive prefix; *total = the sum (same value in every thread).
__device__ __forceinline__ uint32_t block_exscan(uint32_t v, uint32_t nthr, uint32_t bar,
                                                 uint32_t *ws, uint32_t *total) {
    const uint32_t tid = threadIdx.x, lane = tid & 31u, wid = tid >> 5;
    uint32_t incl = v;
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
        uint32_t u = __shfl_up_sync(0xffffffffu, incl, d);
        if (lane >= (uint32_t)d) incl += u;
    }
    if (lane == 31) ws[wid] = incl;
    asm volatile("bar.sync %0, %1;" :: "r"(bar), "r"(nthr) : "memory");
    if (wid == 0) {
        const uint32_t nw = nthr >> 5;
        uint32_t x = lane < nw ? ws[lane] : 0u;
        uint32_t xi = x;
#pragma unroll
        for (int d = 1; d < 32; d <<= 1) {
            uint32_t u = __shfl_up_sync(0xffffffffu, xi, d);
            if (lane >= (uint32_t)d) xi += u;
        }
        if (lane < nw) ws[lane] = xi - x;
        if (lane == 31) ws[32] = xi;
    }
    asm volatile("bar.sync %0, %1;" :: "r"(bar), "r"(nthr) : "memory");
    const uint32_t r = ws[wid] + incl - v;
    *total = ws[32];
    asm volatile("bar.sync %0, %1;" :: "r"(bar), "r"(nthr) : "memory");   // ws reusable
    return r;
}

// Copy the stream bytes [from, to) of job J into shared memory (all nthr threads of the CTA
// take part; the caller synchronises) and return a view of J whose bytes come from there.
// buf + o + (pos - from) holds byte pos, with o chosen so that 16-byte-aligned source addresses
// land on 16-byte-aligned shared addresses (16-byte loads for the bulk of the range).  Needs
// to - from + 16 bytes at buf (16-byte aligned).
__device__ __forceinline__ Job stage_job(const Job &J, uint64_t from, uint64_t to, uint8_t *buf,
                                         int tid, int nthr) {
    const uint32_t o = (uint32_t)((uintptr_t)J.src + (uintptr_t)(from - J.p_begin)) & 15u;
    uint8_t *d = buf + o;                           // d[pos - from] = byte pos
    const uint64_t s0 = from > J.p_begin ? from : J.p_begin;
    for (uint64_t pos = from + tid; pos < to && pos < s0; pos += nthr) d[pos - from] = job_byte(J, pos);
    if (s0 < to) {
        const uintptr_t a0 = (uintptr_t)(J.src + (s0 - J.p_begin));
        const uint64_t a = s0 + (((16u - (a0 & 15u)) & 15u));      // first 16-B-aligned position
        const uint64_t e = a < to ? a + ((to - a) & ~15ull) : a;    // end of the aligned run
        for (uint64_t pos = s0 + tid; pos < to && pos < a; pos += nthr) d[pos - from] = J.src[pos - J.p_begin];
        for (uint64_t pos = e + tid; pos < to; pos += nthr) d[pos - from] = J.src[pos - J.p_begin];
        if (e > a) {
            const uint4 *g = reinterpret_cast<const uint4 *>(J.src + (a - J.p_begin));
            uint4 *sd = reinterpret_cast<uint4 *>(d + (a - from));
            const uint64_t n16 = (e - a) >> 4;
#pragma unroll 4
            for (uint64_t k = tid; k < n16; k += nthr) sd[k] = __ldg(g + k);
        }
    }
    Job V = J;
    V.src = d;
    V.p_begin = from;
    V.prefix = nullptr;
    V.prefix_len = 0;
    return V;
}

// Roll one generic slot into its list; returns the true count.
template <class Tab, bool VEC = true>
__device__ __forceinline__ uint32_t roll_slot(const Job &J, const DevParams &P, const Tab &tab,
                                              uint32_t slot) {
    uint64_t a, b;
    slot_range(J.map, slot, a, b);
    uint32_t cnt = 0;
    uint64_t *lst = J.scratch + (uint64_t)slot * J.cap;
    auto emit = [&](uint64_t c) {
        if (cnt < J.cap) lst[cnt] = c;
        ++cnt;
    };
    roll_generic<Tab, decltype(emit), VEC>(J, P, tab, a, b, emit);
    return cnt;
}

#ifndef SHRED_K1_ONLY   // k1_inst.cu (hot-kernel instances) compiles only k1_bulk
// ------------------------------------------------------------------------------ k1_generic
// Generic-only path: one thread per slot, one group per block of GEN_THREADS slots.
__global__ void __launch_bounds__(GEN_THREADS)
k1_generic(Job J, DevParams P, const GenTables *__restrict__ gt, uint32_t nslots) {
    pdl_entry();
    __shared__ uint64_t sT[256], sU[256];
    __shared__ uint32_t ws[33];
    for (int i = threadIdx.x; i < 256; i += blockDim.x) { sT[i] = gt->T[i]; sU[i] = gt->U[i]; }
    __syncthreads();
    const uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
    SmemGenTab tab{sT, sU};
    const uint32_t cnt = slot < nslots ? roll_slot(J, P, tab, slot) : 0u;
    uint32_t tot;
    const uint32_t off = block_exscan(cnt, GEN_THREADS, 1, ws, &tot);
    if (slot < nslots) { J.counts[slot] = cnt; J.local_off[slot] = off; }
    if (threadIdx.x == 0) J.group_sum[blockIdx.x] = tot;
}

#endif  // SHRED_K1_ONLY

// ------------------------------------------------------------------------------ k1_bulk
// Per-lane constants of the hot loop.  The multipliers are runtime values so that ptxas keeps
// the index math and the marker-test shift on the FMA pipe (IMAD / IMAD.HI) instead of turning
// them into ALU shifts: the ALU pipe is the busiest unit of this loop (ncu r01).
struct BulkCtx {
    uint32_t tab;       // shared address of the T|U image
    uint32_t laneT;     // K63: tab + (lane&15)*8           K32: tab + lane*4
    uint32_t laneU;     // K63: 128 + (lane&15)*8 (byte)     K32: 128 + lane*4 (byte)
    uint32_t mhi;       // K63: 2^(72-k) (t = mulhi(f_hi, mhi))  K40: k-8 (funnel shift)  K32: 2^(40-k)
    uint32_t m256;      // 256 (row stride of the table image)
    uint32_t tmul;      // 2^(32-m): (f_lo * tmul) keeps the low m bits at the top
    uint32_t rsh;       // r << (32-m)
    uint32_t tsel;      // K32B: PRMT selector 0x55s4 placing byte s = (k-8)/8 of f at bits 8..15
    uint32_t tshr, tprod;       // K32T: k - 8, M = Q + 2^k mod 2^32; K63T: k - 40, Q
    uint32_t tprod_hi;          // K63T: 2^(k-32) (the cancel term t << k in the high word)
    uint32_t dm32, r32;         // D - 1 and r as u32 (MK_EQ / MK_LE, D <= 2^32; SHRED_MARK_LOP)
    // MK_DIV (any D = d 2^s, s < 32): f mod D == r  <=>  D | (f + D - r)  (no overflow: f < 2^63,
    // D - r <= 2^63)  <=>  rotr64((f + D - r) * d^-1 mod 2^64, s) <= floor((2^64 - 1) / D)
    uint64_t dc;        // D - r
    uint64_t dinv;      // d^-1 mod 2^64 (d = the odd part of D)
    uint64_t dlim;      // floor((2^64 - 1) / D)
    uint32_t dsh;       // s
    // MK_REM (any other D, either marker set): rem = f - q D with q = floor(f / D) =
    // mulhi64(f, rm) >> rsh2 (Granlund-Montgomery, exact for f < 2^63: rm = ceil(2^(63+l) / D),
    // l = ceil(log2 D), rsh2 = l - 1); marker iff (rem - rlo) mod 2^64 <= rspan
    // ('==': rlo = r, rspan = 0; '<=': rlo = 0, rspan = r).
    uint64_t rm, rd, rlo, rspan;
    uint32_t rsh2;
};

// One byte step, u64 state (deg P = k in 41..63; the paper's reading k = 63), f = fh:fl < 2^k:
//   t = f >> (k-8) = mulhi(fh, 2^(72-k));  f <- (f << 8 mod 2^64) ^ B ^ T[t] ^ U[o]
//   T[t] = (t x^k mod P) ^ ((t << k) mod 2^64) cancels the byte the shift leaves at bits
//   k..k+7 (k = 63: the one bit at 2^63), U[o] = o x^{8w} mod P.  Shift-in by two PRMTs.
// deg 33..40 (FUNNEL): the top byte straddles the two words, t = funnel(fl, fh) >> (k-8).
// The top byte t = f >> (k-8) by SHF on the ALU pipe, not by mulhi: IMAD.HI runs on the
// half-rate fmaheavy pipe, and on the state's dependency chain its latency showed: k63 paper path
// 1,922 -> 1,994 GB/s (k1_bulk, 1 GiB; profiles/r02_k32_ab.txt).  0: IMAD.HI (round 1).
#ifndef SHRED_K63_SHF
#define SHRED_K63_SHF 1
#endif
#ifndef SHRED_K32_SHF
#define SHRED_K32_SHF 1
#endif
#ifndef SHRED_TIDX_LEA
#define SHRED_TIDX_LEA 1  // T row index (t << 8) + lane by LEA (ALU), not IMAD (fmaheavy): k63 1,997 -> 2,005 GB/s
#endif
template <int K, bool FUNNEL = false>
__device__ __forceinline__ void step63(uint32_t &fl, uint32_t &fh, uint32_t in, uint32_t pop,
                                       const BulkCtx &c) {
    const uint32_t t  = FUNNEL ? __funnelshift_rc(fl, fh, c.mhi) : SHRED_K63_SHF ? fh >> c.tshr : __umulhi(fh, c.mhi);
    const uint32_t ti = SHRED_TIDX_LEA ? (t << 8) + c.laneT : t * c.m256 + c.laneT;
    const uint32_t oi = __byte_perm(pop, c.laneU, 0x5504u | (K << 4));
    const uint2 T = lds64(ti);
    const uint2 U = lds64(c.tab + oi);
    const uint32_t nh = __byte_perm(fh, fl, 0x2107u);
    const uint32_t nl = __byte_perm(fl, in, 0x2104u + K);
    fl = nl ^ T.x ^ U.x;
    fh = nh ^ T.y ^ U.y;
}

// One byte step, u32 state (deg P = k in 9..32): t = mulhi(f, 2^(40-k)) = f >> (k-8),
// f <- (f << 8 mod 2^32) ^ B ^ T[t] ^ U[o], T[t] = (t x^k mod P) ^ ((t << k) mod 2^32).
template <int K, bool BYTEIDX>
__device__ __forceinline__ void step32(uint32_t &f, uint32_t in, uint32_t pop, const BulkCtx &c) {
    uint32_t ti;
    if (BYTEIDX)   // deg 16/24/32: t = f >> (k-8) is a whole byte -> one PRMT builds (t << 8) | lane*4
        ti = c.tab + __byte_perm(f, c.laneT - c.tab, c.tsel);
    else
        ti = SHRED_TIDX_LEA ? ((f >> c.tshr) << 8) + c.laneT
                            : (SHRED_K32_SHF ? f >> c.tshr : __umulhi(f, c.mhi)) * c.m256 + c.laneT;
    const uint32_t oi = __byte_perm(pop, c.laneU, 0x5504u | (K << 4));
    const uint32_t T = lds32(ti);
    const uint32_t U = lds32(c.tab + oi);
    f = __byte_perm(f, in, 0x2104u + K) ^ T ^ U;
}

// One byte step, K32T: t = f >> (k-8) (SHF), T = t * M mod 2^32 with M = Q + 2^k mod 2^32 (the
// carry-free product t(x) Q(x) plus the cancel term t << k of the bits the shift leaves at k..31),
// f <- (f << 8 mod 2^32) ^ B ^ T ^ U[o].  The T lookup (and its 29-cycle LDS latency on the
// dependency chain) is gone; only U is looked up.
#ifndef SHRED_K32T_HI
#define SHRED_K32T_HI 0   // 1: t = mulhi(f, 2^(40-k)) on the FMA pipe instead of SHF on the ALU pipe
#endif
template <int K>
__device__ __forceinline__ void step32t(uint32_t &f, uint32_t in, uint32_t pop, const BulkCtx &c) {
    const uint32_t T = (SHRED_K32T_HI ? __umulhi(f, c.mhi) : (f >> c.tshr)) * c.tprod;
    const uint32_t oi = __byte_perm(pop, c.laneU, 0x5504u | (K << 4));
    const uint32_t U = lds32(c.tab + oi);
    f = __byte_perm(f, in, 0x2104u + K) ^ T ^ U;
}

// One byte step, K63T (u64 state, deg k in 41..63): t = f >> (k-8) = fh >> (k-40) (SHF),
// T = (t * 2^(k-32) mod 2^32) : (t * Q) (the carry-free product in the low word, the cancel term
// in the high word), f <- (f << 8 mod 2^64) ^ B ^ T ^ U[o]; U is the only lookup.
#ifndef SHRED_K63T_SHF
#define SHRED_K63T_SHF 1   // A/B: the top byte by IMAD.HI (fmaheavy) instead: 2,227 -> 2,087 GB/s
#endif
template <int K>
__device__ __forceinline__ void step63t(uint32_t &fl, uint32_t &fh, uint32_t in, uint32_t pop,
                                        const BulkCtx &c) {
    const uint32_t t = SHRED_K63T_SHF ? fh >> c.tshr : __umulhi(fh, c.mhi);
    const uint32_t oi = __byte_perm(pop, c.laneU, 0x5504u | (K << 4));
    const uint2 U = lds64(c.tab + oi);
    const uint32_t nh = __byte_perm(fh, fl, 0x2107u);
    const uint32_t nl = __byte_perm(fl, in, 0x2104u + K);
    fl = nl ^ (t * c.tprod) ^ U.x;
    fh = nh ^ (t * c.tprod_hi) ^ U.y;
}

template <int MODE>
struct State;
template <> struct State<MODE_K63T> {
    uint32_t fl = 0, fh = 0;
    __device__ __forceinline__ void set(uint64_t v) { fl = (uint32_t)v; fh = (uint32_t)(v >> 32); }
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step63t<K>(fl, fh, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return fl; }
    __device__ __forceinline__ uint64_t full() const { return ((uint64_t)fh << 32) | fl; }
};
template <> struct State<MODE_K32T> {
    uint32_t f = 0;
    __device__ __forceinline__ void set(uint64_t v) { f = (uint32_t)v; }
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step32t<K>(f, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return f; }
    __device__ __forceinline__ uint64_t full() const { return f; }
};
template <> struct State<MODE_K63> {
    uint32_t fl = 0, fh = 0;
    __device__ __forceinline__ void set(uint64_t v) { fl = (uint32_t)v; fh = (uint32_t)(v >> 32); }
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step63<K>(fl, fh, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return fl; }
    __device__ __forceinline__ uint64_t full() const { return ((uint64_t)fh << 32) | fl; }
};
template <> struct State<MODE_K40> {
    uint32_t fl = 0, fh = 0;
    __device__ __forceinline__ void set(uint64_t v) { fl = (uint32_t)v; fh = (uint32_t)(v >> 32); }
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step63<K, true>(fl, fh, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return fl; }
    __device__ __forceinline__ uint64_t full() const { return ((uint64_t)fh << 32) | fl; }
};
template <> struct State<MODE_K32> {
    uint32_t f = 0;
    __device__ __forceinline__ void set(uint64_t v) { f = (uint32_t)v; }
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step32<K, false>(f, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return f; }
    __device__ __forceinline__ uint64_t full() const { return f; }
};
#ifndef SHRED_K32B_HI
#define SHRED_K32B_HI 0   // 1: K32B builds the T index by IMAD.HI + IMAD (fmaheavy) instead of one PRMT (ALU)
#endif
template <> struct State<MODE_K32B> {
    uint32_t f = 0;
    __device__ __forceinline__ void set(uint64_t v) { f = (uint32_t)v; }
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step32<K, !SHRED_K32B_HI>(f, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return f; }
    __device__ __forceinline__ uint64_t full() const { return f; }
};

// Marker kinds of the hot kernel: MK_EQ / MK_LE: D = 2^m <= 2^32, "fp mod D == r" / "<= r"
// (L447-L451 / L249-L251) on the low word; MK_DIV: "fp mod D == r" for a D that is not a power of
// two (Q8: the integer remainder of the fingerprint's value), on the full state.
// MK_REM: either marker set for any D the other kinds do not take ('<=' with D not a power of two,
// D with 2^32 | D): the remainder itself by a multiply-high division.
enum { MK_EQ = 0, MK_LE = 1, MK_DIV = 2, MK_REM = 3 };
// marker test: (f mod D) == r  <=>  (f_lo << (32-m)) == (r << (32-m))   (D = 2^m <= 2^32)
__device__ __forceinline__ bool is_marker(uint32_t lo, const BulkCtx &c) { return lo * c.tmul == c.rsh; }
// m | BIT if marker else m: ISETP + predicated LOP3 (the PTX predication survives ptxas).
// LE: the "mod D <= r" marker set (L249-L251): (f_lo << (32-m)) <= (r << (32-m)).
// SHRED_MARK_LOP 1: the low m bits by a LOP3 mask (ALU) instead of the IMAD shift (fmaheavy).
// FUSED ('==' only; the u32-state modes): one LOP3 that writes the predicate
// ((lo ^ r) & (D-1)) != 0 (r < D) and no IMAD: 1 ALU op instead of IMAD (fmaheavy) + ISETP (ALU).
// Measured (round 2, 1 GiB k1_bulk, profiles/r02_k32_ab.txt): K32T 2,850 -> 2,960 GB/s, K32 (deg 29)
// 2,602 -> 2,671, K32B 2,778 -> 2,789; the u64-state modes lose 0.6-0.8 % (LSU-bound; IMAD form kept).
// SHRED_MARK_LOP 2 forces the fused form on every mode, -1 on none (A/B).
#ifndef SHRED_MARK_LOP
#define SHRED_MARK_LOP 0
#endif
template <uint32_t BIT, int MK, bool FUSED = false>
__device__ __forceinline__ uint32_t or_if_marker(uint32_t m, uint32_t lo, const BulkCtx &c) {
    if (MK == MK_EQ && SHRED_MARK_LOP != -1 && (FUSED || SHRED_MARK_LOP == 2)) {
        asm("{\n .reg .pred p;\n .reg .b32 t;\n lop3.b32 t, %1, %2, %3, 0x28;\n setp.eq.u32 p, t, 0;\n"
            " @p or.b32 %0, %0, %4;\n}"
            : "+r"(m) : "r"(lo), "r"(c.r32), "r"(c.dm32), "n"(BIT));
        return m;
    }
    const uint32_t x = SHRED_MARK_LOP == 1 ? (lo & c.dm32) : lo * c.tmul;
    const uint32_t y = SHRED_MARK_LOP == 1 ? c.r32 : c.rsh;
    if (MK == MK_LE)
        asm("{\n .reg .pred p;\n setp.le.u32 p, %1, %2;\n @p or.b32 %0, %0, %3;\n}"
            : "+r"(m) : "r"(x), "r"(y), "n"(BIT));
    else
        asm("{\n .reg .pred p;\n setp.eq.u32 p, %1, %2;\n @p or.b32 %0, %0, %3;\n}"
            : "+r"(m) : "r"(x), "r"(y), "n"(BIT));
    return m;
}

// MK_DIV: divisibility of f + D - r by D = d 2^s (Granlund-Montgomery): multiply by d^-1 mod
// 2^64, rotate right by s, compare with floor((2^64 - 1) / D).
template <uint32_t BIT>
__device__ __forceinline__ uint32_t or_if_div(uint32_t m, uint64_t f, const BulkCtx &c) {
    const uint64_t q = (f + c.dc) * c.dinv;
    const uint32_t ql = (uint32_t)q, qh = (uint32_t)(q >> 32);
    const uint64_t rot = ((uint64_t)__funnelshift_r(qh, ql, c.dsh) << 32) | __funnelshift_r(ql, qh, c.dsh);
    return rot <= c.dlim ? (m | BIT) : m;
}

// MK_REM: f mod D by q = mulhi64(f, rm) >> rsh2, rem = f - q D; one window test (rem - rlo) <= rspan.
template <uint32_t BIT>
__device__ __forceinline__ uint32_t or_if_rem(uint32_t m, uint64_t f, const BulkCtx &c) {
    const uint64_t q = __umul64hi(f, c.rm) >> c.rsh2;
    const uint64_t x = f - q * c.rd - c.rlo;
    return x <= c.rspan ? (m | BIT) : m;
}

// MK_REM, u32 state (deg <= 32, f < 2^32, so D <= 2^32 and MK_REM has D < 2^32, l <= 32): the
// same quotient from two 32x32 -> 64 products, h = (f rm) >> 32 = f rm_hi + hi32(f rm_lo) and
// q = hi32(h) >> (l - 1); rem < 2^32, so the rest runs in 32 bits.
template <uint32_t BIT>
__device__ __forceinline__ uint32_t or_if_rem32(uint32_t m, uint32_t f, const BulkCtx &c) {
    const uint64_t h = (uint64_t)f * (uint32_t)(c.rm >> 32) + __umulhi(f, (uint32_t)c.rm);
    const uint32_t q = (uint32_t)(h >> 32) >> c.rsh2;
    const uint32_t x = f - q * (uint32_t)c.rd - (uint32_t)c.rlo;
    return x <= (uint32_t)c.rspan ? (m | BIT) : m;
}

struct SlotOut {
    uint64_t *lst; uint32_t cnt; uint32_t cap;
};

// Emit the marker hits of one 16-byte chunk: bit j of m = a hit at window end pos + j.
static __device__ __noinline__ void emit_mask(uint32_t m, uint64_t pos, uint64_t min_i, uint64_t c_limit,
                                       SlotOut &o) {
    while (m) {
        const int j = __ffs(m) - 1;
        m &= m - 1;
        const uint64_t i = pos + (uint64_t)j;
        if (i >= min_i && i + 1 < c_limit) {
            if (o.cnt < o.cap) o.lst[o.cnt] = i + 1;
            ++o.cnt;
        }
    }
}

// One word (4 bytes) of CH interleaved chains; hit bits accumulate into m[ch] (bit 4J+q).
// PACKM: with two chains per thread the hit bits of both share one register (chain 1 at bits
// 16..31), so a chunk costs one mask init (SEL) and one "any hit" test for the pair instead of
// one each per chain (ALU-pipe ops: the u32-state kernels are ALU-bound).
#ifndef SHRED_PACKM
#define SHRED_PACKM 1
#endif
template <int CH> struct Pack { static constexpr bool on = SHRED_PACKM && CH == 2; };
#if SHRED_HITMODE == 0
#define SHRED_MARK(ch, q) m[ch] |= is_marker(st[ch].low(), c) ? (1u << (4 * J + q)) : 0u;
#else
// the hit test of position 4J+Q for every chain, chain index CHI a compile-time constant (the
// hit bit is an immediate operand of the predicated add)
template <int MODE, int CH, int J, int Q, int MK, int CHI = 0>
__device__ __forceinline__ void mark_chains(State<MODE> (&st)[CH], uint32_t (&m)[CH], const BulkCtx &c) {
    if constexpr (CHI < CH) {
        constexpr int MI = Pack<CH>::on ? 0 : CHI;
        constexpr uint32_t BIT = 1u << (4 * J + Q + (Pack<CH>::on ? 16 * CHI : 0));
        constexpr bool U32 = MODE == MODE_K32 || MODE == MODE_K32B || MODE == MODE_K32T;
        if constexpr (MK == MK_DIV)
            m[MI] = or_if_div<BIT>(m[MI], st[CHI].full(), c);
        else if constexpr (MK == MK_REM && U32)
            m[MI] = or_if_rem32<BIT>(m[MI], st[CHI].low(), c);
        else if constexpr (MK == MK_REM)
            m[MI] = or_if_rem<BIT>(m[MI], st[CHI].full(), c);
        else
            m[MI] = or_if_marker<BIT, MK, U32>(m[MI], st[CHI].low(), c);
        mark_chains<MODE, CH, J, Q, MK, CHI + 1>(st, m, c);
    }
}
#define SHRED_MARK(ch, q) if (ch == 0) mark_chains<MODE, CH, J, q, MK>(st, m, c);
#endif
template <int MODE, int CH, bool TEST, int J, int MK>
__device__ __forceinline__ void word4xN(State<MODE> (&st)[CH], const uint32_t (&in)[CH],
                                        const uint32_t (&pop)[CH], uint32_t (&m)[CH], const BulkCtx &c) {
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) st[ch].template step<0>(in[ch], pop[ch], c);
    if (TEST) {
#pragma unroll
        for (int ch = 0; ch < CH; ++ch) { SHRED_MARK(ch, 0) }
    }
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) st[ch].template step<1>(in[ch], pop[ch], c);
    if (TEST) {
#pragma unroll
        for (int ch = 0; ch < CH; ++ch) { SHRED_MARK(ch, 1) }
    }
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) st[ch].template step<2>(in[ch], pop[ch], c);
    if (TEST) {
#pragma unroll
        for (int ch = 0; ch < CH; ++ch) { SHRED_MARK(ch, 2) }
    }
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) st[ch].template step<3>(in[ch], pop[ch], c);
    if (TEST) {
#pragma unroll
        for (int ch = 0; ch < CH; ++ch) { SHRED_MARK(ch, 3) }
    }
}
#undef SHRED_MARK

// 16 bytes of CH chains in one basic block (ILP across the chains): d = data chunk,
// p = the chunk 48 bytes earlier (its bytes leave the window).
template <int MODE, int CH, bool TEST, int MK>
__device__ __forceinline__ void chunk16xN(State<MODE> (&st)[CH], const uint4 (&d)[CH], const uint4 (&p)[CH],
                                          const BulkCtx &c, uint32_t (&m)[CH]) {
    uint32_t in[CH], po[CH];
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) m[ch] = 0;
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) { in[ch] = d[ch].x; po[ch] = p[ch].x; }
    word4xN<MODE, CH, TEST, 0, MK>(st, in, po, m, c);
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) { in[ch] = d[ch].y; po[ch] = p[ch].y; }
    word4xN<MODE, CH, TEST, 1, MK>(st, in, po, m, c);
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) { in[ch] = d[ch].z; po[ch] = p[ch].z; }
    word4xN<MODE, CH, TEST, 2, MK>(st, in, po, m, c);
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) { in[ch] = d[ch].w; po[ch] = p[ch].w; }
    word4xN<MODE, CH, TEST, 3, MK>(st, in, po, m, c);
}

struct BulkConst {
    uint32_t mhi, m256, tmul, rsh, tsel;
    uint32_t tshr, tprod;      // K32T / K63T (BulkCtx)
    uint32_t tprod_hi;         // K63T (BulkCtx)
    uint32_t dm32, r32;        // BulkCtx
    uint64_t dc, dinv, dlim;   // MK_DIV constants (BulkCtx)
    uint32_t dsh;
    uint64_t rm, rd, rlo, rspan;   // MK_REM constants (BulkCtx)
    uint32_t rsh2;
    const uint64_t *pos;       // DIRECT_WARM: C_j[b] = b x^{8j} mod P at pos[256 j + b], j < w
    uint32_t w;                // window bytes (DIRECT_WARM)
    uint32_t fu, fsel;  // FN windows (w % 16 != 0): e = 16*ceil(w/16) - w = 4*fu + v, fsel = PRMT
                        // selector of bytes v..v+3 (0x3210 + 0x1111 v)
    uint32_t wa;        // ceil(w/16): the long-window mode's warm-up chunks and pop distance
};

// The 16 bytes leaving the window at chunk q are bytes [16(q-A) + e, +16), A = WCH = ceil(w/16),
// e = 16A - w: chunk q-A itself (w a multiple of 16), else a byte funnel of chunks q-A (lo) and
// q-A+1 (hi) at the uniform offset e (one switch per chunk for every chain, 4 PRMTs per chain).
template <bool FN, int CH>
__device__ __forceinline__ void pops16(const uint4 (&lo)[CH], const uint4 (&hi)[CH], uint4 (&p)[CH],
                                       const BulkConst &K) {
    if (!FN) {
#pragma unroll
        for (int ch = 0; ch < CH; ++ch) p[ch] = lo[ch];
        return;
    }
#define SHRED_FUN(a, b, c, d, e)                                                              \
    for (int ch = 0; ch < CH; ++ch) {                                                        \
        const uint32_t C[8] = {lo[ch].x, lo[ch].y, lo[ch].z, lo[ch].w, hi[ch].x, hi[ch].y, hi[ch].z, hi[ch].w}; \
        p[ch] = make_uint4(__byte_perm(C[a], C[b], K.fsel), __byte_perm(C[b], C[c], K.fsel),  \
                           __byte_perm(C[c], C[d], K.fsel), __byte_perm(C[d], C[e], K.fsel)); \
    }
    switch (K.fu) {
        case 0: SHRED_FUN(0, 1, 2, 3, 4) break;
        case 1: SHRED_FUN(1, 2, 3, 4, 5) break;
        case 2: SHRED_FUN(2, 3, 4, 5, 6) break;
        default: SHRED_FUN(3, 4, 5, 6, 7) break;
    }
#undef SHRED_FUN
}

// The hot kernel.  blockDim = NTC consumers + 1 producer warp; one CTA per SM.
// blockIdx < nc: bulk CTA, rows blockIdx*ROWS + tid + ch*NTC (ch < CH); blockIdx == nc: the
// edge CTA.  Rounds of ROUND = 64/CH bytes per row arrive in a SHRED_STAGES-deep TMA ring (the 8 lanes
// of a quarter warp read 8 consecutive rows' 16-byte chunks from 8 distinct bank groups:
// SWIZZLE_32B for 32-byte rounds, no swizzle for 16-byte rounds).  The window is fixed at
// w = 48 = 3 chunks of 16 B: the byte leaving the window at chunk q is the same byte slot of
// chunk q-3, kept in a 4-slot register ring per chain (slot = chunk index mod 4).  WCH = w/16
// (w in {16, 32, 48, 64}) generalises the pop distance; MK selects the marker kind.
template <int MODE, class C, int WCH, int MK, bool FN = false>
__global__ void __launch_bounds__(C::NTC + 32, 1)
k1_bulk(const __grid_constant__ CUtensorMap tmap, const __grid_constant__ CUtensorMap tmap_pop,
        const uint4 *__restrict__ tab_img, const GenTables *__restrict__ gt, Job J, DevParams P, BulkConst K) {
    constexpr bool LW = WCH == 0;                    // long window (w > 64): pops from a TMA tile
    constexpr int BAR_OFF = LW ? LwLayout<C>::BAR_OFF : C::BAR_OFF;
    if (SHRED_PDL_EARLY) pdl_trigger(); else pdl_entry();
    constexpr int CH = C::CH, NTC = C::NTC, ROUND = C::ROUND, CPR = C::CPR;
    extern __shared__ uint8_t smem_raw[];
    // align the dynamic shared base to 1 KiB (the TMA swizzle pattern is address-based)
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    const uint32_t sbase = smem_u32(smem);
    const uint32_t stages = sbase + TAB_BYTES;
    const uint32_t bars = sbase + BAR_OFF;         // full[s] at +8s, empty[s] at +64+8s
    uint32_t *ws = reinterpret_cast<uint32_t *>(smem + BAR_OFF + 128);
    const uint32_t popst = stages + STAGES * C::STAGE;       // LW: the pop tiles
    const int tid = threadIdx.x;

    if (blockIdx.x == J.map.nc) {                    // ---- edge CTA: head + tail, generic loop
        uint64_t *sT = reinterpret_cast<uint64_t *>(smem + TAB_BYTES);
        uint64_t *sU = sT + 256;
        for (int i = tid; i < 256; i += blockDim.x) { sT[i] = gt->T[i]; sU[i] = gt->U[i]; }
        if (SHRED_PDL_EARLY) pdl_wait();
        // Stage the head and tail byte ranges (with their w-1 warm-up bytes) in the idle stage
        // ring, so the byte loop reads shared memory instead of one dependent global load per
        // byte (that latency chain set a ~16 us floor on every call).
        uint8_t *buf = smem + TAB_BYTES + 4096;
        const uint64_t cap = (uint64_t)STAGES * C::STAGE - 4096;
        const uint64_t warm = (uint64_t)P.w - 1u, lo = J.p_begin - J.prefix_len;
        const uint64_t hf = J.map.head_start >= lo + warm ? J.map.head_start - warm : lo;
        const uint64_t tf = J.map.tail_start >= lo + warm ? J.map.tail_start - warm : lo;
        const uint64_t hl = J.map.n_head ? J.map.b0 - hf : 0, tl = J.map.n_tail ? J.map.t_end - tf : 0;
        const uint64_t hsz = (hl + 31u) & ~15ull;       // + alignment slack, 16-B multiple
        const bool sh = hl && hsz <= cap, stl = tl && hsz + tl + 16u <= cap;
        Job JH = J, JT = J;
        if (sh) JH = stage_job(J, hf, J.map.b0, buf, tid, blockDim.x);
        if (stl) JT = stage_job(J, tf, J.map.t_end, buf + hsz, tid, blockDim.x);
        __syncthreads();
        if (tid >= NTC) return;
        SmemGenTab tab{sT, sU};
        const uint32_t tail0 = J.map.n_head + J.map.nrows;
        // staged segments (shared memory): byte loads; unstaged (too long to stage): vector loads
        const uint32_t ch = (uint32_t)tid < J.map.n_head
                                ? (sh ? roll_slot<SmemGenTab, false>(JH, P, tab, tid) : roll_slot(JH, P, tab, tid)) : 0u;
        const uint32_t ct = (uint32_t)tid < J.map.n_tail
                                ? (stl ? roll_slot<SmemGenTab, false>(JT, P, tab, tail0 + tid) : roll_slot(JT, P, tab, tail0 + tid)) : 0u;
        uint32_t th, tt;
        const uint32_t oh = block_exscan(ch, NTC, 1, ws, &th);
        const uint32_t ot = block_exscan(ct, NTC, 1, ws, &tt);
        if ((uint32_t)tid < J.map.n_head) { J.counts[tid] = ch; J.local_off[tid] = oh; }
        if ((uint32_t)tid < J.map.n_tail) { J.counts[tail0 + tid] = ct; J.local_off[tail0 + tid] = ot; }
        if (tid == 0) { J.group_sum[0] = th; J.group_sum[J.map.nc + 1] = tt; }
        return;
    }

    // the 64 KiB T|U image arrives by TMA bulk copies (tabbar), overlapping the set-up below
    const uint32_t tabbar = bars + 120;
    if (tid == 0) {
        for (int s = 0; s < STAGES; ++s) {
            mbar_init(bars + 8 * s, 1);
            mbar_init(bars + 64 + 8 * s, NTC / 32);
        }
        mbar_init(tabbar, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
        mbar_expect_tx(tabbar, TAB_BYTES);
#pragma unroll
        for (int q = 0; q < 4; ++q)
            bulk_g2s(sbase + q * (TAB_BYTES / 4), reinterpret_cast<const uint8_t *>(tab_img) + q * (TAB_BYTES / 4),
                     TAB_BYTES / 4, tabbar);
    }
    if (SHRED_PDL_EARLY) pdl_wait();
    __syncthreads();

    const uint32_t row0 = blockIdx.x * C::ROWS;
    const uint32_t nrounds = (uint32_t)(J.map.S / ROUND);     // S % 32 == 0: a loop iteration (RPI
                                                              // rounds = 64 B) may end half way

    if (tid >= NTC) {                                // ---- producer warp
        if (tid == NTC) {
            for (uint32_t r = 0; r < nrounds; ++r) {
                const uint32_t s = r % STAGES;
                if (r >= STAGES) mbar_wait_sleep(bars + 64 + 8 * s, ((r / STAGES) - 1u) & 1u);
                mbar_expect_tx(bars + 8 * s, LW ? C::STAGE + LwLayout<C>::POP_STAGE : C::STAGE);
                const uint32_t dst = stages + s * C::STAGE;
#pragma unroll
                for (int q = 0; q < C::ROWS / C::BOX; ++q)
                    tma_load_2d(dst + q * C::BOX * ROUND, &tmap, (int)(r * ROUND), (int)(row0 + q * C::BOX),
                                bars + 8 * s);
                if (LW) {
                    const uint32_t pd = popst + s * LwLayout<C>::POP_STAGE;
#pragma unroll
                    for (int q = 0; q < C::ROWS / C::BOX; ++q)
                        tma_load_2d(pd + q * C::BOX * LW_POPW, &tmap_pop, (int)(r * ROUND), (int)(row0 + q * C::BOX),
                                    bars + 8 * s);
                }
            }
        }
        return;
    }

    // ---- consumers: thread tid owns rows row0 + tid + ch*NTC
    const int lane = tid & 31;
    BulkCtx c;
    c.tab = sbase;
    if (MODE == MODE_K63 || MODE == MODE_K40 || MODE == MODE_K63T) {
        c.laneT = sbase + (uint32_t)(lane & 15) * 8u;
        c.laneU = 128u + (uint32_t)(lane & 15) * 8u;
    } else {
        c.laneT = sbase + (uint32_t)lane * 4u;
        c.laneU = 128u + (uint32_t)lane * 4u;
    }
    c.mhi = K.mhi; c.m256 = K.m256; c.tmul = K.tmul; c.rsh = K.rsh; c.tsel = K.tsel;
    c.tshr = K.tshr; c.tprod = K.tprod; c.tprod_hi = K.tprod_hi; c.dm32 = K.dm32; c.r32 = K.r32;
    c.dc = K.dc; c.dinv = K.dinv; c.dlim = K.dlim; c.dsh = K.dsh;
    c.rm = K.rm; c.rd = K.rd; c.rlo = K.rlo; c.rspan = K.rspan; c.rsh2 = K.rsh2;

    bool act[CH];
    uint64_t pos0[CH];
    SlotOut o[CH];
    State<MODE> st[CH];
    uint4 R[CH][4];                                   // ring: slot q = chunk index mod 4
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) {
        const uint32_t row = row0 + tid + ch * NTC;
        act[ch] = row < J.map.nrows;
        pos0[ch] = J.map.b0 + (uint64_t)row * J.map.S;
        o[ch].lst = J.scratch + (uint64_t)(J.map.n_head + row) * J.cap;
        SHRED_ASSERT(!act[ch] || J.map.n_head + row < J.map.n_head + J.map.nrows);
        o[ch].cnt = 0; o[ch].cap = J.cap;
    }
    {
        // warm-up: the 16*WCH bytes before each row, from a zero state (the plan keeps them inside
        // src: b0 >= p_begin + 16*WCH).  A row at the very start of a stream (no carry) finds
        // virtual zero bytes before p_begin instead: zero bytes pushed into a zero state leave it
        // zero (T[0] = U[0] = 0), and only full windows are tested (min_i).  The ring slots of
        // the 4 - WCH chunks not rolled stay zero.
        const uint4 Z = make_uint4(0, 0, 0, 0);
#pragma unroll
        for (int ch = 0; ch < CH; ++ch) {
#pragma unroll
            for (int q = 0; q < 4; ++q) R[ch][q] = Z;
            if (act[ch]) {
#pragma unroll
                for (int q = (C::DIRECT_WARM ? 0 : 4 - WCH); q < 4; ++q) {
                    // chunk q holds stream bytes [pos0 - 64 + 16q, +16): inside the job's bytes?
                    if (pos0[ch] + 16u * (uint32_t)q >= J.p_begin + 64u)
                        R[ch][q] = __ldg(reinterpret_cast<const uint4 *>(J.src + (pos0[ch] + 16u * (uint32_t)q - 64u - J.p_begin)));
                }
            }
        }
        if (C::DIRECT_WARM) {
            // The state at the row start is the fingerprint of the w bytes before it (the rolled
            // warm-up pushes 64 bytes and pops all but the last w): XOR of C_j[B[pos0-1-j]] over
            // j < w, independent loads (no T|U lookups: the table TMA is still in flight).
#pragma unroll
            for (int ch = 0; ch < CH; ++ch) {
                uint64_t f = 0;
#pragma unroll
                for (int j = 0; j < 64; ++j) {
                    if ((uint32_t)j < K.w) {
                        const int i = 63 - j;             // byte pos0-1-j = byte i of R[ch][0..3]
                        const uint4 v = R[ch][i >> 4];
                        const uint32_t wd = ((i >> 2) & 3) == 0 ? v.x : ((i >> 2) & 3) == 1 ? v.y
                                          : ((i >> 2) & 3) == 2 ? v.z : v.w;
                        f ^= __ldg(K.pos + 256 * j + ((wd >> (8 * (i & 3))) & 0xFFu));
                    }
                }
                st[ch].set(f);
            }
        }
        mbar_wait(tabbar, 0);                         // T|U image resident
        uint32_t m[CH];
#pragma unroll
        for (int q = (C::DIRECT_WARM ? 4 : 4 - WCH); q < 4; ++q) {
            // chunks before 4 - WCH were never pushed: their bytes pop as zero
            uint4 d[CH], p[CH];
            uint4 lo[CH], hi[CH];
#pragma unroll
            for (int ch = 0; ch < CH; ++ch) {
                d[ch] = R[ch][q];
                lo[ch] = (q - WCH >= 4 - WCH) ? R[ch][q - WCH] : Z;
                hi[ch] = (q + 1 - WCH >= 4 - WCH) ? R[ch][q + 1 - WCH] : Z;
            }
            pops16<FN, CH>(lo, hi, p, K);
            chunk16xN<MODE, CH, false, MK>(st, d, p, c, m);
        }
        if (LW) {
            // long window: roll the 16*wa bytes before the row (inside src: the plan keeps b0 >=
            // p_begin + 16*wa) from a zero state.  Their pops lie before the warm-up start
            // (virtual zeros), except in the last chunk: bytes [16 - e, 16) of its pops are the
            // warm-up's first e bytes (e = 16*wa - w), i.e. the funnel of (zero, first chunk).
            uint4 first[CH], nxt[CH];
            auto wload = [&](int ch, uint32_t k) {     // warm-up chunk k of chain ch
                SHRED_ASSERT(!act[ch] || (pos0[ch] >= J.p_begin + 16ull * K.wa &&
                                          pos0[ch] + 16ull * k + 16u <= J.map.t_end + 16ull * K.wa));
                return act[ch] ? __ldg(reinterpret_cast<const uint4 *>(
                                     J.src + (pos0[ch] - 16ull * K.wa + 16ull * k - J.p_begin)))
                               : Z;
            };
#pragma unroll
            for (int ch = 0; ch < CH; ++ch) nxt[ch] = wload(ch, 0);
            for (uint32_t k = 0; k < K.wa; ++k) {
                uint4 d[CH], p[CH];
#pragma unroll
                for (int ch = 0; ch < CH; ++ch) {
                    d[ch] = nxt[ch];                     // the next chunk's load overlaps this one's steps
                    if (k + 1 < K.wa) nxt[ch] = wload(ch, k + 1);
                    if (k == 0) first[ch] = d[ch];
                }
                if (k + 1 == K.wa) {
                    uint4 zl[CH];
#pragma unroll
                    for (int ch = 0; ch < CH; ++ch) zl[ch] = Z;
                    pops16<FN, CH>(zl, first, p, K);
                } else {
#pragma unroll
                    for (int ch = 0; ch < CH; ++ch) p[ch] = Z;
                }
                chunk16xN<MODE, CH, false, MK>(st, d, p, c, m);
            }
        }
    }

    // TMA swizzle of the 16-byte chunk index (rows of ROUND bytes; tid + ch*NTC has the same
    // low bits as tid): SWIZZLE_64B: ^ (row >> 1) & 3, SWIZZLE_32B: ^ (row >> 2) & 1, 16 B: none
    const uint32_t swz = (ROUND == 64) ? (((uint32_t)tid >> 1) & 3u)
                       : (ROUND == 32) ? (((uint32_t)tid >> 2) & 1u) : 0u;
    for (uint32_t r = 0; r < nrounds; r += C::RPI) {
#pragma unroll
        for (int qr = 0; qr < C::RPI; ++qr) {             // round r + qr: chunks qr*CPR .. +CPR-1
            if (qr > 0 && r + qr >= nrounds) break;       // rows of an odd number of 32-byte rounds
            const uint32_t s = (r + qr) % STAGES;
            mbar_wait(bars + 8 * s, ((r + qr) / STAGES) & 1u);
            const uint32_t sb = stages + s * C::STAGE;
            uint4 D[CH][CPR];
#pragma unroll
            for (int ch = 0; ch < CH; ++ch)
#pragma unroll
                for (int u = 0; u < CPR; ++u)
                    D[ch][u] = lds128(sb + (uint32_t)(tid + ch * NTC) * ROUND + (((uint32_t)u ^ swz) << 4));
            // LW: the round's pop chunks (aligned, 16*wa bytes behind) and the next one (funnel)
            uint4 PQ[CH][LW ? CPR + 1 : 1];
            if (LW) {
                const uint32_t pb = popst + s * LwLayout<C>::POP_STAGE;
#pragma unroll
                for (int ch = 0; ch < CH; ++ch)
#pragma unroll
                    for (int u = 0; u < (LW ? CPR + 1 : 1); ++u)
                        if (u < CPR || FN) PQ[ch][u] = lds128(pb + (uint32_t)(tid + ch * NTC) * LW_POPW + 16u * u);
                if (FN && r + qr + 1 == nrounds) {
                    // the last round's funnel chunk lies past the pop tile's rows (zero fill): the
                    // same bytes from global memory (the row's own data, 16*wa - S + ... behind)
#pragma unroll
                    for (int ch = 0; ch < CH; ++ch)
                        if (act[ch]) {
                            SHRED_ASSERT(pos0[ch] + (uint64_t)nrounds * ROUND <= J.map.b0 + (uint64_t)J.map.nrows * J.map.S &&
                                         pos0[ch] + (uint64_t)nrounds * ROUND >= J.p_begin + 16ull * K.wa);
                            PQ[ch][CPR] = __ldg(reinterpret_cast<const uint4 *>(
                                J.src + (pos0[ch] + (uint64_t)nrounds * ROUND - 16ull * K.wa - J.p_begin)));
                        }
                }
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(bars + 64 + 8 * s);
#pragma unroll
            for (int u = 0; u < CPR; ++u) {
                const int cq = qr * CPR + u;          // chunk index mod 4 (compile time)
                uint4 d[CH], p[CH];
                uint32_t m[CH];
#pragma unroll
                for (int ch = 0; ch < CH; ++ch) { d[ch] = D[ch][u]; }
                {
                    uint4 lo[CH], hi[CH];
#pragma unroll
                    for (int ch = 0; ch < CH; ++ch) {
                        if (LW) {
                            lo[ch] = PQ[ch][u];
                            hi[ch] = PQ[ch][LW ? u + 1 : 0];
                        } else {
                            lo[ch] = R[ch][(cq + 4 - WCH) & 3];
                            hi[ch] = (WCH == 1) ? D[ch][u] : R[ch][(cq + 5 - WCH) & 3];
                        }
                    }
                    pops16<FN, CH>(lo, hi, p, K);
                }
                chunk16xN<MODE, CH, true, MK>(st, d, p, c, m);
#pragma unroll
                for (int ch = 0; ch < CH; ++ch) R[ch][cq] = D[ch][u];
                // rows past nrows (TMA zero fill; only in the last CTA) are tested only once a
                // chunk has a hit (zero windows are markers when r = 0 or '<='): one "any hit"
                // test per chunk for the pair of chains
                if (Pack<CH>::on) {
                    if (m[0]) {
#pragma unroll
                        for (int ch = 0; ch < CH; ++ch) {
                            const uint32_t mc = (m[0] >> (16 * ch)) & 0xFFFFu;
                            if (mc && act[ch])
                                emit_mask(mc, pos0[ch] + (uint64_t)(r + qr) * ROUND + 16u * u, J.min_i, J.c_limit, o[ch]);
                        }
                    }
                } else {
#pragma unroll
                    for (int ch = 0; ch < CH; ++ch)
                        if (m[ch] && act[ch])
                            emit_mask(m[ch], pos0[ch] + (uint64_t)(r + qr) * ROUND + 16u * u, J.min_i, J.c_limit, o[ch]);
                }
            }
        }
    }
    uint32_t base = 0;
#pragma unroll
    for (int ch = 0; ch < CH; ++ch) {
        uint32_t tot;
        const uint32_t off = block_exscan(act[ch] ? o[ch].cnt : 0u, NTC, 1, ws, &tot);
        if (act[ch]) {
            const uint32_t slot = J.map.n_head + row0 + tid + ch * NTC;
            J.counts[slot] = o[ch].cnt;
            J.local_off[slot] = base + off;
        }
        base += tot;
    }
    if (tid == 0) J.group_sum[1 + blockIdx.x] = base;
}

// A hot-kernel instance; pick_k1 / pick_k1_small (k1_inst.cu) map parameters to instances.
typedef void (*K1Fn)(const __grid_constant__ CUtensorMap, const __grid_constant__ CUtensorMap, const uint4 *,
                     const GenTables *, Job, DevParams, BulkConst);
K1Fn pick_k1(int k, bool byteidx, int wch, int mk, bool fn, bool tprod = false);
K1Fn pick_k1_small(int k, bool byteidx, int wch, int mk, bool fn, bool tprod = false);

#ifndef SHRED_K1_ONLY
// ------------------------------------------------------------------------------ k_total
// Sum of the group sums -> aux->total (bounded path: needed on the host before k_scatter).
__global__ void k_total(const uint64_t *__restrict__ group_sum, uint32_t ngroups, Aux *aux) {
    pdl_entry();
    uint64_t s = 0;
    for (uint32_t g = threadIdx.x; g < ngroups; g += blockDim.x) s += group_sum[g];
    for (int d = 16; d; d >>= 1) s += __shfl_xor_sync(0xffffffffu, s, d);
    __shared__ uint64_t w[32];
    if ((threadIdx.x & 31) == 0) w[threadIdx.x >> 5] = s;
    __syncthreads();
    if (threadIdx.x == 0) {
        uint64_t t = 0;
        for (uint32_t i = 0; i < (blockDim.x + 31) / 32; ++i) t += w[i];
        aux->total = t;
    }
}

// ------------------------------------------------------------------------------ k_scatter
// One thread per slot (blocks of 256).  Every block scans the group sums itself (<= a few
// hundred) to get its groups' bases; offset(slot) = base(group) + local_off[slot].
// dst index = (streaming ? aux->out_pos + aux->held : 0) + offset.  Block 0 writes the
// total (aux->total, and *n_direct with the overflow flag if given).  Overflowed slots re-roll.
constexpr int SCATTER_THREADS = 256;
constexpr int MAX_GROUPS = 4096;
__global__ void __launch_bounds__(SCATTER_THREADS)
k_scatter(Job J, DevParams P, const GenTables *__restrict__ gt, uint32_t nslots,
          uint64_t *__restrict__ dst, uint64_t dst_cap, Aux *aux, int streaming,
          uint64_t *n_direct, int reset) {
    pdl_entry();
    __shared__ uint64_t gbase[MAX_GROUPS];
    __shared__ uint64_t wsum[SCATTER_THREADS / 32 + 1];
    const uint32_t ng = J.map.ngroups;
    const uint32_t tid = threadIdx.x;
    // This slot's count, local offset and first two list entries do not depend on the group scan:
    // issue their loads first so their latency overlaps the scan (the kernel is a short chain of
    // dependent global accesses; ~0.4 candidates per slot at D = 8 KiB).
    const uint32_t slot = blockIdx.x * blockDim.x + tid;
    uint32_t cnt = 0, loff = 0;
    uint64_t l0 = 0, l1 = 0;
    const uint64_t *lst = J.scratch + (uint64_t)slot * J.cap;
    if (slot < nslots) {
        cnt = J.counts[slot];
        loff = J.local_off[slot];
        if (cnt >= 1 && cnt <= J.cap) l0 = lst[0];
        if (cnt >= 2 && cnt <= J.cap) l1 = lst[1];
    }
    // exclusive scan of group_sum[0..ng) into gbase (chunks of 256 with a running carry)
    uint64_t carry = 0;
    for (uint32_t b = 0; b < ng; b += SCATTER_THREADS) {
        const uint32_t g = b + tid;
        const uint64_t v = g < ng ? J.group_sum[g] : 0ull;
        uint64_t incl = v;
        for (int d = 1; d < 32; d <<= 1) {
            uint64_t u = __shfl_up_sync(0xffffffffu, incl, d);
            if ((tid & 31) >= (uint32_t)d) incl += u;
        }
        if ((tid & 31) == 31) wsum[tid >> 5] = incl;
        __syncthreads();
        if (tid == 0) {
            uint64_t r = 0;
            for (int w = 0; w < SCATTER_THREADS / 32; ++w) { uint64_t x = wsum[w]; wsum[w] = r; r += x; }
            wsum[SCATTER_THREADS / 32] = r;
        }
        __syncthreads();
        if (g < ng) gbase[g] = carry + wsum[tid >> 5] + incl - v;
        carry += wsum[SCATTER_THREADS / 32];
        __syncthreads();
    }
    const uint64_t total = carry;
    if (blockIdx.x == 0 && tid == 0) {
        if (reset) {                          // a one-shot bounded call: its size-rule state (no
            aux->s = 0; aux->held = 0;         // block reads it here: streaming == 0)
            aux->held_val = 0; aux->out_pos = 0;
        }
        aux->total = total;
        aux->ncand = total;
        aux->dense = total > dst_cap ? 1ull : 0ull;
        if (n_direct) { *n_direct = total; if (total > dst_cap) aux->overflow = 1; }
    }
    if (slot >= nslots || cnt == 0) return;
    const uint64_t off = gbase[slot_group(J.map, slot)] + loff;
    const uint64_t base = (streaming ? aux->out_pos + aux->held : 0ull) + off;
    if (cnt <= J.cap) {
        if (base < dst_cap) dst[base] = l0;
        if (cnt >= 2 && base + 1 < dst_cap) dst[base + 1] = l1;
        for (uint32_t j = 2; j < cnt; ++j)
            if (base + j < dst_cap) dst[base + j] = lst[j];
        if (off + cnt == total) aux->last_cand = cnt == 1 ? l0 : cnt == 2 ? l1 : lst[cnt - 1];
    } else {
        uint64_t a, b;
        slot_range(J.map, slot, a, b);
        uint64_t k = 0, last = 0;
        GlobalGenTab tab{gt};
        roll_generic(J, P, tab, a, b, [&](uint64_t c) {
            if (base + k < dst_cap) dst[base + k] = c;
            ++k; last = c;
        });
        if (off + cnt == total) aux->last_cand = last;
    }
}

// ------------------------------------------------------------------------------ streaming glue
// After an unbounded piece ending at `end`: emit the previously held cut at out_pos, hold the
// piece's last candidate if it sits exactly at the stream end, advance out_pos.
__global__ void k_piece_done(Aux *aux, uint64_t *dst, uint64_t dst_cap, uint64_t end) {
    pdl_entry();
    if (threadIdx.x != 0 || blockIdx.x != 0) return;
    const uint64_t held = aux->held;
    if (held && aux->out_pos < dst_cap) dst[aux->out_pos] = aux->held_val;
    const uint64_t tot = aux->total;
    const int hold_new = (tot > 0 && aux->last_cand == end);
    aux->out_pos += held + tot - (uint64_t)hold_new;
    aux->held = (uint64_t)hold_new;
    aux->held_val = hold_new ? end : 0;
}

__global__ void k_call_begin(Aux *aux) {
    pdl_entry();
    aux->out_pos = 0;
}

__global__ void k_call_end(Aux *aux, uint64_t *n_out, uint64_t cap, volatile uint64_t *sticky_flag) {
    pdl_entry();
    *n_out = aux->out_pos;
    if (aux->out_pos > cap) {
        aux->overflow = 1;
        if (sticky_flag) *sticky_flag = 1;
    }
}

__global__ void k_stream_reset(Aux *aux) {
    pdl_entry();
    aux->total = 0; aux->last_cand = 0; aux->out_pos = 0;
    aux->s = 0; aux->held = 0; aux->held_val = 0; aux->dense = 0;
}

// A piece with no window ends: no candidates (the count the size rule reads, the dense flag and
// the caller's count if given).
__global__ void k_no_slots(Aux *aux, uint64_t *n_direct, int reset) {
    pdl_entry();
    if (reset) { aux->s = 0; aux->held = 0; aux->held_val = 0; aux->out_pos = 0; }
    aux->total = 0; aux->ncand = 0; aux->dense = 0;
    if (n_direct) *n_direct = 0;
}

__global__ void k_write_u64(uint64_t *p, uint64_t v) {
    pdl_entry();
    *p = v;
}

// Entry / exit of shred_size_bound_state.
__global__ void k_state_in(Aux *aux, uint64_t s, uint64_t held) {
    pdl_entry();
    aux->total = 0; aux->last_cand = 0; aux->out_pos = 0; aux->dense = 0;
    aux->s = s; aux->held = held; aux->held_val = held ? s : 0;
}
__global__ void k_state_in_dev(Aux *aux, const uint64_t *state) {
    pdl_entry();
    const uint64_t s = state[0], held = state[1] ? 1ull : 0ull;
    aux->total = 0; aux->last_cand = 0; aux->out_pos = 0; aux->dense = 0;
    aux->s = s; aux->held = held; aux->held_val = held ? s : 0;
}
__global__ void k_state_out(const Aux *aux, uint64_t *state, uint64_t *n_out, uint64_t cap) {
    pdl_entry();
    state[0] = aux->s; state[1] = aux->held;
    *n_out = aux->out_pos;
}

// New carry = the last min(keep, old_len + len) bytes of (old carry || src[0..len)).
__global__ void k_carry(const uint8_t *old_c, uint32_t old_len, const uint8_t *src, uint64_t len,
                        uint8_t *new_c, uint32_t keep) {
    pdl_entry();
    const uint64_t tot = (uint64_t)old_len + len;
    const uint32_t nl = (uint32_t)(tot < keep ? tot : keep);
    for (uint32_t j = threadIdx.x; j < nl; j += blockDim.x) {
        const uint64_t v = tot - nl + j;        // index into (old || src)
        new_c[j] = (v < old_len) ? old_c[v] : src[v - old_len];
    }
}

// ------------------------------------------------------------------------------ synth fill
// Counter-mode SplitMix64: word k of stream seed is
// mix(seed + (k+1) * 0x9E3779B97F4A7C15), little-endian at bytes 8k..8k+7.
__device__ __forceinline__ uint64_t splitmix_word(uint64_t seed, uint64_t k) {
    uint64_t z = seed + (k + 1ull) * 0x9E3779B97F4A7C15ull;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}
__global__ void k_synth_fill(uint8_t *dst, uint64_t len, uint64_t seed, uint64_t offset) {
    pdl_entry();
    // byte j of dst = byte (offset + j) of the stream; each thread writes 16 bytes
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x * 16ull;
    for (uint64_t j0 = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) * 16ull; j0 < len; j0 += stride) {
        const uint64_t p = offset + j0;
        const uint64_t kw = p >> 3;
        const uint32_t sh = (uint32_t)(p & 7u);
        const uint64_t w0 = splitmix_word(seed, kw), w1 = splitmix_word(seed, kw + 1),
                       w2 = splitmix_word(seed, kw + 2);
        uint8_t buf[24];
#pragma unroll
        for (int q = 0; q < 8; ++q) {
            buf[q] = (uint8_t)(w0 >> (8 * q));
            buf[8 + q] = (uint8_t)(w1 >> (8 * q));
            buf[16 + q] = (uint8_t)(w2 >> (8 * q));
        }
        const uint64_t m = (len - j0) < 16 ? (len - j0) : 16;
        if (m == 16 && (((uintptr_t)(dst + j0)) & 15u) == 0) {
            uint4 v;
            uint8_t *vb = reinterpret_cast<uint8_t *>(&v);
#pragma unroll
            for (int q = 0; q < 16; ++q) vb[q] = buf[sh + q];
            *reinterpret_cast<uint4 *>(dst + j0) = v;
        } else {
            for (uint64_t q = 0; q < m; ++q) dst[j0 + q] = buf[sh + q];
        }
    }
}
#endif  // SHRED_K1_ONLY

}  // namespace shred

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
//   k1_bulk<MODE>   TMA-staged hot loop.  One thread = one row of S bytes of the input viewed
//                   as a 2-D [rows][S] tensor; rounds of 64 B per row arrive in a 4-stage
//                   shared-memory ring (SWIZZLE_64B, conflict-free LDS.128).  T/U live in
//                   shared memory, replicated per lane so the data-dependent lookups never
//                   bank-conflict.  A per-16-byte predicate detects the rare marker hit;
//                   hits replay that chunk exactly and append c to the thread's slot list.
//   k1_generic      Any valid parameters, byte at a time; also the head/tail of fast paths.
//   k_scan          Exclusive scan of per-slot candidate counts (one CTA).
//   k_scatter       Ordered compaction of the per-slot lists into the destination; slots
//                   that overflowed their list re-roll their range and write directly.
//   k_size_bound    The sequential min/max rule (one warp), with streaming state.
#pragma once
#include <cstdint>
#include <cuda.h>
#include <cuda_runtime.h>

namespace shred {

enum { MODE_K63 = 1, MODE_K32 = 2, MODE_GENERIC = 3 };

constexpr int NT          = 512;               // consumer threads (rows) per CTA
constexpr int ROUND       = 64;                // bytes per row per pipeline round
constexpr int STAGES      = 4;                 // TMA ring depth
constexpr int BOX_ROWS    = 256;               // rows per TMA box (hardware max 256)
constexpr int TAB_BYTES   = 65536;             // replicated T|U image (256 rows x 256 B)
constexpr int STAGE_BYTES = NT * ROUND;        // 32 KiB
constexpr int BAR_OFFSET  = TAB_BYTES + STAGES * STAGE_BYTES;
constexpr int BULK_SMEM   = BAR_OFFSET + 1024; // + barriers; + 1 KiB so the base can be aligned
constexpr int GEN_THREADS = 256;

// Slot id -> range of window-end positions.  Slots are numbered in stream order:
// [0, n_head) generic head segments, then the bulk rows, then generic tail segments.
struct SlotMap {
    uint64_t head_start; uint64_t head_seg; uint32_t n_head;
    uint32_t nrows;      uint64_t b0;       uint64_t S;
    uint64_t tail_start; uint64_t tail_seg; uint32_t n_tail;
    uint64_t t_end;
};

struct DevParams {              // chunking parameters as the kernels need them
    uint64_t dmask;             // D - 1
    uint64_t magic;             // r
    uint64_t kmask;             // 2^k - 1
    uint32_t k;                 // deg P
    uint32_t w;                 // window bytes
};

struct Job {
    const uint8_t *src;         // src[0] is stream position p_begin
    uint64_t p_begin;
    const uint8_t *prefix;      // virtual bytes [p_begin - prefix_len, p_begin) (the carry)
    uint32_t prefix_len;
    uint32_t cap;               // per-slot list capacity
    uint64_t min_i;             // w - 1: only full windows are tested (reading Q10)
    uint64_t c_limit;           // emit c only if c < c_limit (reading Q11)
    uint32_t *counts;           // [nslots] true candidate count per slot
    uint64_t *scratch;          // [nslots * cap] per-slot candidate lists
    SlotMap map;
};

struct GenTables { uint64_t T[256]; uint64_t U[256]; };

// Device-resident streaming / output state (one per ctx).
struct Aux {
    uint64_t total;             // candidates of the current piece (k_scan)
    uint64_t last_cand;         // last candidate of the current piece (k_scatter)
    uint64_t out_pos;           // cuts already written by the current API call
    uint64_t s;                 // size rule: last cut (absolute)
    uint64_t held;              // 1 if a cut at exactly the previous stream end is held
    uint64_t held_val;
    uint64_t overflow;          // sticky: an output did not fit
    uint64_t pad;
};

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

// Roll the exact fingerprint over window ends [seg_start, seg_end) from a zero state
// w-1 bytes earlier (or the first available byte), calling emit(c) for every candidate.
// Plain byte-at-a-time form: f <- ((f << 8) mod x^k) ^ b ^ T[top byte] ^ U[B[pos-w]].
template <class Tab, class Emit>
__device__ __forceinline__ void roll_generic(const Job &J, const DevParams &P, const Tab &tab,
                                             uint64_t seg_start, uint64_t seg_end, Emit emit) {
    const uint64_t lo = J.p_begin - J.prefix_len;
    const uint64_t warm = (uint64_t)P.w - 1u;
    uint64_t p = (seg_start >= lo + warm) ? seg_start - warm : lo;
    uint64_t f = 0;
    for (uint64_t pos = p; pos < seg_end; ++pos) {
        uint32_t b = job_byte(J, pos);
        uint32_t t = (uint32_t)(f >> (P.k - 8u)) & 0xFFu;
        f = ((f << 8) & P.kmask) ^ (uint64_t)b ^ tab.T(t);
        if (pos >= p + P.w) f ^= tab.U(job_byte(J, pos - P.w));
        if (pos >= seg_start && pos >= J.min_i && (f & P.dmask) == P.magic && pos + 1 < J.c_limit)
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

// ------------------------------------------------------------------------------ k1_generic
// One thread per generic slot (head slots, then tail slots).
__global__ void __launch_bounds__(GEN_THREADS)
k1_generic(Job J, DevParams P, const GenTables *__restrict__ gt) {
    __shared__ uint64_t sT[256], sU[256];
    for (int i = threadIdx.x; i < 256; i += blockDim.x) { sT[i] = gt->T[i]; sU[i] = gt->U[i]; }
    __syncthreads();
    const uint32_t g = blockIdx.x * blockDim.x + threadIdx.x;
    const uint32_t ngen = J.map.n_head + J.map.n_tail;
    if (g >= ngen) return;
    const uint32_t slot = (g < J.map.n_head) ? g : g + J.map.nrows;
    uint64_t a, b;
    slot_range(J.map, slot, a, b);
    uint32_t cnt = 0;
    uint64_t *lst = J.scratch + (uint64_t)slot * J.cap;
    SmemGenTab tab{sT, sU};
    roll_generic(J, P, tab, a, b, [&](uint64_t c) {
        if (cnt < J.cap) lst[cnt] = c;
        ++cnt;
    });
    J.counts[slot] = cnt;
}

// ------------------------------------------------------------------------------ k1_bulk
struct BulkCtx {
    uint32_t tab;       // shared address of the T|U image
    uint32_t laneT;     // K63: tab + (lane&15)*8           K32: lane*4
    uint32_t laneU;     // K63: 128 + (lane&15)*8 (byte)     K32: 128 + lane*4 (byte)
    uint32_t mask, magic;
};

// One byte step, K63 (deg P = 63, fully reduced u64 state f = fh:fl, f < 2^63):
//   t = f >> 55;  f <- (f << 8 mod 2^64) ^ B ^ T[t] ^ U[o]
//   T[t] = (t x^63 mod P) ^ ((t & 1) << 63) cancels the bit the shift leaves at 2^63,
//   U[o] = o x^{8w} mod P.   Shift-in by two byte permutes (PRMT).
template <int K>
__device__ __forceinline__ void step63(uint32_t &fl, uint32_t &fh, uint32_t in, uint32_t pop,
                                       const BulkCtx &c) {
    const uint32_t t  = fh >> 23;
    const uint32_t ti = t * 256u + c.laneT;
    const uint32_t oi = __byte_perm(pop, c.laneU, 0x5504u | (K << 4));
    const uint2 T = lds64(ti);
    const uint2 U = lds64(c.tab + oi);
    const uint32_t nh = __byte_perm(fh, fl, 0x2107u);
    const uint32_t nl = __byte_perm(fl, in, 0x2104u + K);
    fl = nl ^ T.x ^ U.x;
    fh = nh ^ T.y ^ U.y;
}

// One byte step, K32 (deg P = 32, u32 state): f <- (f << 8) ^ B ^ T[f >> 24] ^ U[o].
template <int K>
__device__ __forceinline__ void step32(uint32_t &f, uint32_t in, uint32_t pop, const BulkCtx &c) {
    const uint32_t ti = __byte_perm(f, c.laneT, 0x5534u);
    const uint32_t oi = __byte_perm(pop, c.laneU, 0x5504u | (K << 4));
    const uint32_t T = lds32(c.tab + ti);
    const uint32_t U = lds32(c.tab + oi);
    f = __byte_perm(f, in, 0x2104u + K) ^ T ^ U;
}

template <int MODE>
struct State;
template <> struct State<MODE_K63> {
    uint32_t fl = 0, fh = 0;
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step63<K>(fl, fh, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return fl; }
};
template <> struct State<MODE_K32> {
    uint32_t f = 0;
    template <int K> __device__ __forceinline__ void step(uint32_t in, uint32_t pop, const BulkCtx &c) {
        step32<K>(f, in, pop, c);
    }
    __device__ __forceinline__ uint32_t low() const { return f; }
};

// 4 bytes of one word: hit |= (low bits of the fingerprint after each byte == r).
template <int MODE, bool TEST>
__device__ __forceinline__ void word4(State<MODE> &s, uint32_t in, uint32_t pop, const BulkCtx &c,
                                      bool &hit) {
    s.template step<0>(in, pop, c); if (TEST) hit |= ((s.low() & c.mask) == c.magic);
    s.template step<1>(in, pop, c); if (TEST) hit |= ((s.low() & c.mask) == c.magic);
    s.template step<2>(in, pop, c); if (TEST) hit |= ((s.low() & c.mask) == c.magic);
    s.template step<3>(in, pop, c); if (TEST) hit |= ((s.low() & c.mask) == c.magic);
}

struct SlotOut {
    uint64_t *lst; uint32_t cnt; uint32_t cap;
    uint64_t min_i, c_limit;
    __device__ __forceinline__ void emit(uint64_t i) {       // i = window end position
        if (i >= min_i && i + 1 < c_limit) {
            if (cnt < cap) lst[cnt] = i + 1;
            ++cnt;
        }
    }
};

// Replay one 16-byte chunk from its saved entry state, emitting every marker hit exactly.
template <int MODE>
__device__ __noinline__ void replay_chunk(State<MODE> s, uint4 d, uint4 p, uint64_t pos,
                                          const BulkCtx &c, SlotOut &o) {
    const uint32_t dw[4] = {d.x, d.y, d.z, d.w};
    const uint32_t pw[4] = {p.x, p.y, p.z, p.w};
#pragma unroll
    for (int j = 0; j < 4; ++j) {
        s.template step<0>(dw[j], pw[j], c); if ((s.low() & c.mask) == c.magic) o.emit(pos + 4 * j + 0);
        s.template step<1>(dw[j], pw[j], c); if ((s.low() & c.mask) == c.magic) o.emit(pos + 4 * j + 1);
        s.template step<2>(dw[j], pw[j], c); if ((s.low() & c.mask) == c.magic) o.emit(pos + 4 * j + 2);
        s.template step<3>(dw[j], pw[j], c); if ((s.low() & c.mask) == c.magic) o.emit(pos + 4 * j + 3);
    }
}

template <int MODE, bool TEST>
__device__ __forceinline__ void chunk16(State<MODE> &s, const uint4 &d, const uint4 &p, uint64_t pos,
                                        const BulkCtx &c, SlotOut &o) {
    const State<MODE> s0 = s;
    bool hit = false;
    word4<MODE, TEST>(s, d.x, p.x, c, hit);
    word4<MODE, TEST>(s, d.y, p.y, c, hit);
    word4<MODE, TEST>(s, d.z, p.z, c, hit);
    word4<MODE, TEST>(s, d.w, p.w, c, hit);
    if (TEST && hit) replay_chunk<MODE>(s0, d, p, pos, c, o);
}

// The hot kernel.  blockDim = NT consumers + 1 producer warp; one CTA per SM.
// The window is fixed at w = 48 = 3 chunks of 16 B: the byte leaving the window at chunk q
// is the same byte slot of chunk q-3, kept in registers (R1..R3 = chunks 1..3 of the
// previous round).
template <int MODE>
__global__ void __launch_bounds__(NT + 32, 1)
k1_bulk(const __grid_constant__ CUtensorMap tmap, const uint4 *__restrict__ tab_img, Job J,
        uint32_t mask, uint32_t magic) {
    extern __shared__ uint8_t smem_raw[];
    // align the dynamic shared base to 1 KiB (SWIZZLE_64B pattern is address-based)
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    const uint32_t sbase = smem_u32(smem);
    const uint32_t stages = sbase + TAB_BYTES;
    const uint32_t bars = sbase + BAR_OFFSET;      // full[s] at +8s, empty[s] at +64+8s
    const int tid = threadIdx.x;

    for (int i = tid; i < TAB_BYTES / 16; i += blockDim.x)
        reinterpret_cast<uint4 *>(smem)[i] = tab_img[i];
    if (tid == 0) {
        for (int s = 0; s < STAGES; ++s) {
            mbar_init(bars + 8 * s, 1);
            mbar_init(bars + 64 + 8 * s, NT / 32);
        }
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    }
    __syncthreads();

    const uint32_t row0 = blockIdx.x * NT;
    const uint32_t nrounds = (uint32_t)(J.map.S / ROUND);

    if (tid >= NT) {                                 // ---- producer warp
        if (tid == NT) {
            for (uint32_t r = 0; r < nrounds; ++r) {
                const uint32_t s = r % STAGES;
                if (r >= STAGES) mbar_wait(bars + 64 + 8 * s, ((r / STAGES) - 1u) & 1u);
                mbar_expect_tx(bars + 8 * s, STAGE_BYTES);
                const uint32_t dst = stages + s * STAGE_BYTES;
                tma_load_2d(dst, &tmap, (int)(r * ROUND), (int)row0, bars + 8 * s);
                tma_load_2d(dst + BOX_ROWS * ROUND, &tmap, (int)(r * ROUND), (int)(row0 + BOX_ROWS),
                            bars + 8 * s);
            }
        }
        return;
    }

    // ---- consumers: thread tid owns row row0 + tid
    const int lane = tid & 31;
    const uint32_t row = row0 + tid;
    const bool active = row < J.map.nrows;
    const uint64_t rpos = J.map.b0 + (uint64_t)row * J.map.S;

    BulkCtx c;
    c.tab = sbase;
    if (MODE == MODE_K63) {
        c.laneT = sbase + (uint32_t)(lane & 15) * 8u;
        c.laneU = 128u + (uint32_t)(lane & 15) * 8u;
    } else {
        c.laneT = (uint32_t)lane * 4u;
        c.laneU = 128u + (uint32_t)lane * 4u;
    }
    c.mask = mask; c.magic = magic;
    SlotOut o;
    const uint32_t slot = J.map.n_head + row;
    o.lst = J.scratch + (uint64_t)slot * J.cap;
    o.cnt = 0; o.cap = J.cap; o.min_i = J.min_i; o.c_limit = J.c_limit;

    State<MODE> st;
    uint4 R1 = make_uint4(0, 0, 0, 0), R2 = R1, R3 = R1;
    if (active) {
        // warm-up: the 64 bytes before the row (b0 >= p_begin + 64 guarantees they are in src)
        const uint4 *h = reinterpret_cast<const uint4 *>(J.src + (rpos - 64u - J.p_begin));
        const uint4 H0 = __ldg(h + 0), H1 = __ldg(h + 1), H2 = __ldg(h + 2), H3 = __ldg(h + 3);
        const uint4 Z = make_uint4(0, 0, 0, 0);
        chunk16<MODE, false>(st, H0, Z, 0, c, o);
        chunk16<MODE, false>(st, H1, Z, 0, c, o);
        chunk16<MODE, false>(st, H2, Z, 0, c, o);
        chunk16<MODE, false>(st, H3, H0, 0, c, o);
        R1 = H1; R2 = H2; R3 = H3;
    }

    const uint32_t sw = ((uint32_t)tid >> 1) & 3u;
    const uint32_t rowoff = (uint32_t)tid * ROUND;
    for (uint32_t r = 0; r < nrounds; ++r) {
        const uint32_t s = r % STAGES;
        mbar_wait(bars + 8 * s, (r / STAGES) & 1u);
        const uint32_t rb = stages + s * STAGE_BYTES + rowoff;
        const uint4 D0 = lds128(rb + ((0u ^ sw) << 4));
        const uint4 D1 = lds128(rb + ((1u ^ sw) << 4));
        const uint4 D2 = lds128(rb + ((2u ^ sw) << 4));
        const uint4 D3 = lds128(rb + ((3u ^ sw) << 4));
        __syncwarp();
        if (lane == 0) mbar_arrive(bars + 64 + 8 * s);
        if (active) {
            const uint64_t pos = rpos + (uint64_t)r * ROUND;
            chunk16<MODE, true>(st, D0, R1, pos + 0, c, o);
            chunk16<MODE, true>(st, D1, R2, pos + 16, c, o);
            chunk16<MODE, true>(st, D2, R3, pos + 32, c, o);
            chunk16<MODE, true>(st, D3, D0, pos + 48, c, o);
        }
        R1 = D1; R2 = D2; R3 = D3;
    }
    if (active) J.counts[slot] = o.cnt;
}

// ------------------------------------------------------------------------------ k_scan
// Exclusive scan of counts[0..n) -> offsets (u64); total -> aux->total (and *n_direct if set).
__global__ void __launch_bounds__(1024)
k_scan(const uint32_t *__restrict__ counts, uint32_t n, uint64_t *__restrict__ offsets, Aux *aux,
       uint64_t *n_direct, uint64_t direct_cap) {
    __shared__ uint64_t warp_sums[32];
    const uint32_t tid = threadIdx.x;
    const uint32_t per = (n + blockDim.x - 1) / blockDim.x;
    const uint32_t a = tid * per;
    const uint32_t b = min(n, a + per);
    uint64_t sum = 0;
    for (uint32_t i = a; i < b; ++i) sum += counts[i];
    // block-wide exclusive scan of `sum`
    uint64_t incl = sum;
    for (int d = 1; d < 32; d <<= 1) {
        uint64_t v = __shfl_up_sync(0xffffffffu, incl, d);
        if ((tid & 31) >= (uint32_t)d) incl += v;
    }
    if ((tid & 31) == 31) warp_sums[tid >> 5] = incl;
    __syncthreads();
    if (tid < 32) {
        uint64_t v = warp_sums[tid];
        uint64_t vi = v;
        for (int d = 1; d < 32; d <<= 1) {
            uint64_t u = __shfl_up_sync(0xffffffffu, vi, d);
            if (tid >= (uint32_t)d) vi += u;
        }
        warp_sums[tid] = vi - v;                  // exclusive warp prefix
    }
    __syncthreads();
    uint64_t run = warp_sums[tid >> 5] + incl - sum;
    for (uint32_t i = a; i < b; ++i) { offsets[i] = run; run += counts[i]; }
    if (tid == blockDim.x - 1) {
        aux->total = run;
        if (n_direct) {
            *n_direct = run;
            if (run > direct_cap) aux->overflow = 1;
        }
    }
}

// ------------------------------------------------------------------------------ k_scatter
// One thread per slot.  dst[base + offsets[slot] + j] for j < count (bounded by dst_cap);
// base = aux->out_pos + aux->held when `streaming`, else 0.  Overflowed slots re-roll.
__global__ void __launch_bounds__(256)
k_scatter(Job J, DevParams P, const GenTables *__restrict__ gt, uint32_t nslots,
          const uint64_t *__restrict__ offsets, uint64_t *__restrict__ dst, uint64_t dst_cap,
          Aux *aux, int streaming) {
    const uint32_t slot = blockIdx.x * blockDim.x + threadIdx.x;
    if (slot >= nslots) return;
    const uint32_t cnt = J.counts[slot];
    if (cnt == 0) return;
    const uint64_t base = (streaming ? aux->out_pos + aux->held : 0ull) + offsets[slot];
    const uint64_t total = aux->total;
    if (cnt <= J.cap) {
        const uint64_t *lst = J.scratch + (uint64_t)slot * J.cap;
        for (uint32_t j = 0; j < cnt; ++j)
            if (base + j < dst_cap) dst[base + j] = lst[j];
        if (offsets[slot] + cnt == total) aux->last_cand = lst[cnt - 1];
    } else {
        uint64_t a, b;
        slot_range(J.map, slot, a, b);
        uint64_t k = 0, last = 0;
        GlobalGenTab tab{gt};
        roll_generic(J, P, tab, a, b, [&](uint64_t c) {
            if (base + k < dst_cap) dst[base + k] = c;
            ++k; last = c;
        });
        if (offsets[slot] + cnt == total) aux->last_cand = last;
    }
}

// ------------------------------------------------------------------------------ streaming glue
// After an unbounded piece ending at `end`: emit the previously held cut at out_pos, hold the
// piece's last candidate if it sits exactly at the stream end, advance out_pos.
__global__ void k_piece_done(Aux *aux, uint64_t *dst, uint64_t dst_cap, uint64_t end) {
    if (threadIdx.x != 0 || blockIdx.x != 0) return;
    const uint64_t held = aux->held;
    if (held && aux->out_pos < dst_cap) dst[aux->out_pos] = aux->held_val;
    const uint64_t tot = aux->total;
    const int hold_new = (tot > 0 && aux->last_cand == end);
    aux->out_pos += held + tot - (uint64_t)hold_new;
    aux->held = (uint64_t)hold_new;
    aux->held_val = hold_new ? end : 0;
}

__global__ void k_call_begin(Aux *aux) { aux->out_pos = 0; }

__global__ void k_call_end(Aux *aux, uint64_t *n_out, uint64_t cap, volatile uint64_t *sticky_flag) {
    *n_out = aux->out_pos;
    if (aux->out_pos > cap) {
        aux->overflow = 1;
        if (sticky_flag) *sticky_flag = 1;
    }
}

__global__ void k_stream_reset(Aux *aux) {
    aux->total = 0; aux->last_cand = 0; aux->out_pos = 0;
    aux->s = 0; aux->held = 0; aux->held_val = 0;
}

__global__ void k_write_u64(uint64_t *p, uint64_t v) { *p = v; }

// New carry = the last min(keep, old_len + len) bytes of (old carry || src[0..len)).
__global__ void k_carry(const uint8_t *old_c, uint32_t old_len, const uint8_t *src, uint64_t len,
                        uint8_t *new_c, uint32_t keep) {
    const uint64_t tot = (uint64_t)old_len + len;
    const uint32_t nl = (uint32_t)(tot < keep ? tot : keep);
    for (uint32_t j = threadIdx.x; j < nl; j += blockDim.x) {
        const uint64_t v = tot - nl + j;        // index into (old || src)
        new_c[j] = (v < old_len) ? old_c[v] : src[v - old_len];
    }
}

// ------------------------------------------------------------------------------ k_size_bound
// The min/max rule (readings Q12-Q15), one warp, sequential over the
// ascending candidates; lanes load 32 candidates at a time.  State (s, held) lives in `aux`.
//   final = 1 (one-shot): stream end N = end; cuts must be < N.
//   final = 0 (streaming piece): a cut exactly at `end` is held (emitted by the next piece).
// ncand is read from *ncand_dev if non-null, else ncand_host.
__global__ void __launch_bounds__(32)
k_size_bound(const uint64_t *__restrict__ cand, const uint64_t *ncand_dev, uint64_t ncand_host,
             uint64_t end, int final_, uint64_t minsz, uint64_t maxsz,
             uint64_t *__restrict__ dst, uint64_t dst_cap, Aux *aux) {
    const int lane = threadIdx.x;
    const uint64_t n = ncand_dev ? *ncand_dev : ncand_host;
    uint64_t s = aux->s;
    uint64_t k = aux->out_pos;
    uint64_t held = aux->held, held_val = aux->held_val;
    if (held) { if (lane == 0 && k < dst_cap) dst[k] = held_val; ++k; held = 0; }
    const uint64_t INF = ~0ull;
    const uint64_t mx = maxsz ? maxsz : INF;
    for (uint64_t b = 0; b < n; b += 32) {
        const uint64_t v = (b + lane < n) ? cand[b + lane] : 0ull;
        const int m = (int)((n - b) < 32 ? (n - b) : 32);
        for (int j = 0; j < m; ++j) {
            const uint64_t c = __shfl_sync(0xffffffffu, v, j);
            if (maxsz) {
                while (c - s > mx) { s += mx; if (lane == 0 && k < dst_cap) dst[k] = s; ++k; }
            }
            if (c - s >= minsz) {
                s = c;
                if (!final_ && c == end) { held = 1; held_val = c; }
                else { if (lane == 0 && k < dst_cap) dst[k] = c; ++k; }
            }
        }
    }
    if (maxsz) {
        while (end - s > mx) { s += mx; if (lane == 0 && k < dst_cap) dst[k] = s; ++k; }
    }
    if (lane == 0) {
        aux->s = s; aux->out_pos = k; aux->held = held; aux->held_val = held_val;
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

}  // namespace shred

// shred.cu — host side of the C ABI declared in include/shred.h.
//
// Owns: parameter validation (incl. an irreducibility test of div(x)),
// host construction of the push/pop tables, the per-ctx device buffers, the launch sequence
//   K1 (k1_bulk TMA hot loop + its edge CTA | k1_generic) -> k_scatter [-> sb_* size rule]
// and the host-fed streaming ring (§4.1-§4.2: pinned buffers, async H2D on a copy
// stream, double/triple buffering of device slots).  No CPU fallback: every step of the path
// runs in the kernels of kernels.cuh.
#include "kernels.cuh"
#include "size_bound.cuh"
#include "sha256.cuh"
#include "dedup.cuh"

#ifndef SHRED_HASH_NOPDL
// k_hash_chunks is launched plainly, not as a programmatic dependent: launched early (during
// k_hash_scatter) its 148 one-warp-per-SMSP CTAs were placed wherever the scatter left room,
// several on some SMs and none on others, and the 1 GiB hash took 4.6-5.6 ms instead of 3.7
// (profiles/r02_hash_ab.txt).  Its launch latency is negligible against milliseconds of hashing.
#define SHRED_HASH_NOPDL 1
#endif
#ifndef SHRED_HASH_WS
#define SHRED_HASH_WS 1   // one buffer: k_hash_chunks_ws (0: k_hash_chunks, A/B)
#endif
#ifndef SHRED_HASH_WS_BATCH
#define SHRED_HASH_WS_BATCH 1   // batches too (0: k_hash_chunks, 2 CTAs per SM, A/B)
#endif
#ifndef SHRED_HASH_CTAS_PER_SM
#define SHRED_HASH_CTAS_PER_SM 1
#endif
#ifndef SHRED_HASH_THREADS
#define SHRED_HASH_THREADS 128                // one warp per SM sub-partition
#endif
#include "../../include/shred.h"

#include <cstdarg>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <string>
#include <vector>

using namespace shred;

// ============================================================================ GF(2) on the host
// Polynomials over GF(2) in a u64 (bit t = coefficient of x^t).  Used only to build tables.
namespace {

int deg64(uint64_t p) { return p ? 63 - __builtin_clzll(p) : -1; }

// a * x mod P  (deg a < k, P of degree k <= 63)
inline uint64_t mulx(uint64_t a, uint64_t P, int k) {
    a <<= 1;
    if ((a >> k) & 1u) a ^= P;
    return a;
}
// a * b mod P, Horner over the bits of b from the top
uint64_t mulmod(uint64_t a, uint64_t b, uint64_t P, int k) {
    uint64_t acc = 0;
    for (int t = k - 1; t >= 0; --t) {
        acc = mulx(acc, P, k);
        if ((b >> t) & 1u) acc ^= a;
    }
    return acc;
}
uint64_t gcd2(uint64_t a, uint64_t b) {
    while (b) {
        while (a && deg64(a) >= deg64(b)) a ^= b << (deg64(a) - deg64(b));
        std::swap(a, b);
    }
    return a;
}
// Ben-Or: P of degree k is irreducible iff gcd(x^(2^i) - x mod P, P) = 1 for i = 1..k/2.
bool irreducible(uint64_t P) {
    const int k = deg64(P);
    if (k < 1) return false;
    uint64_t xp = 2u;                    // x^(2^0) = x  (k >= 2 here)
    if (k == 1) return true;
    for (int i = 1; i <= k / 2; ++i) {
        xp = mulmod(xp, xp, P, k);       // x^(2^i)
        if (gcd2(P, xp ^ 2u) != 1u) return false;
    }
    return true;
}
// t(x) * x^e mod P for every byte t, via the 8 basis values x^(e+j) mod P.
void byte_times_xpow(uint64_t P, int k, uint64_t e, uint64_t out[256]) {
    uint64_t xe = 1u;                    // x^0
    for (uint64_t n = 0; n < e; ++n) xe = mulx(xe, P, k);
    uint64_t basis[8];
    for (int j = 0; j < 8; ++j) { basis[j] = xe; xe = mulx(xe, P, k); }
    for (int t = 0; t < 256; ++t) {
        uint64_t v = 0;
        for (int j = 0; j < 8; ++j) if ((t >> j) & 1) v ^= basis[j];
        out[t] = v;
    }
}

#ifndef SHRED_L2PROMO
#define SHRED_L2PROMO CU_TENSOR_MAP_L2_PROMOTION_L2_128B   // TMA L2 promotion of the row tiles (A/B: r01_ab_variants)
#endif
#ifndef SHRED_PDL
#define SHRED_PDL 1       // 0: plain stream serialization (A/B)
#endif
#ifndef SHRED_EDGE_GS
#define SHRED_EDGE_GS 16  // edge-CTA head/tail segment: each is a chain of w-1 + GS dependent steps
#endif
#ifndef SHRED_TPROD
#define SHRED_TPROD 1     // MODE_K32T for eligible polynomials (0: table modes only, A/B)
#endif
#ifndef SHRED_BYTEIDX
#define SHRED_BYTEIDX 1   // deg 8/16/24/32: PRMT table index (MODE_K32B); 0: IMAD index (MODE_K32)
#endif
typedef CUresult (*EncodeTiledFn)(CUtensorMap *, CUtensorMapDataType, cuuint32_t, void *,
                                  const cuuint64_t *, const cuuint64_t *, const cuuint32_t *,
                                  const cuuint32_t *, CUtensorMapInterleave, CUtensorMapSwizzle,
                                  CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

const char *kErr[] = {"ok", "invalid argument", "out of memory", "CUDA error",
                      "invalid stream state", "output capacity exceeded (sticky)"};

}  // namespace

// ============================================================================ ctx
struct shred_ctx {
    shred_params p{};
    int device = 0;
    int path = 0;
    int mode = MODE_GENERIC;             // kernels.cuh MODE_* of the hot kernel instance
    int k = 0;
    int mk = MK_EQ;                      // marker kind of the hot kernel (kernels.cuh MK_*)
    DevParams dp{};
    uint4 *d_tab_img = nullptr;          // 64 KiB replicated T|U image (fast paths)
    GenTables *d_gen = nullptr;          // plain T/U (generic path, recompute)
    uint64_t *d_pos = nullptr;           // positional tables C_j[b] = b x^{8j} mod P, j < w (small shape)
    EncodeTiledFn encode = nullptr;
    CUtensorMap tm_cache;                // the last encoded tensor map and its key (plan_job)
    uint64_t tm_key[4] = {0, 0, 0, 0};
    bool tm_valid = false;
    K1Fn k1_fn = nullptr;                // the hot-kernel instance for these parameters
    int k1_smem = 0;                     // its dynamic shared memory
    K1Fn k1_small_fn = nullptr;          // the same with the small-input shape (or null)
    int sm_count = 148;

    // scratch (grown on demand, synchronously)
    uint32_t *d_counts = nullptr; uint64_t counts_cap = 0;
    uint32_t *d_local = nullptr; uint64_t local_cap = 0;
    uint64_t *d_groups = nullptr; uint64_t groups_cap = 0;
    uint64_t *d_scratch = nullptr; uint64_t scratch_cap = 0;   // in u64 entries
    uint64_t *d_cand = nullptr; uint64_t cand_cap = 0;         // bounded mode ordered list
    uint64_t *d_sb = nullptr; uint64_t sb_cap = 0;             // size-rule block scratch
    Aux *d_aux = nullptr;                // [0] one-shot calls, [1] the stream
    uint64_t *h_pinned = nullptr;        // small pinned readback area
    unsigned long long *d_queue = nullptr;   // work queue of k_hash_chunks
    uint32_t *d_hhist = nullptr;             // k_hash_* length buckets
    uint32_t *d_order = nullptr; uint64_t order_cap = 0;   // length-sorted chunk order
    DedupTable index{};                  // f3: device hash set of digests (shred_index_*)
    uint64_t *h_flag = nullptr;          // mapped pinned word: a streaming call overflowed
    uint64_t *d_flag = nullptr;          // its device alias

    // streaming state (host mirror)
    uint64_t pos = 0;                    // bytes fed so far
    uint8_t *d_carry[2] = {nullptr, nullptr};
    int carry_idx = 0;
    uint32_t carry_len = 0;
    int sticky = SHRED_OK;
    int ring_n = 2; uint64_t ring_bytes = 256ull << 20;
    std::vector<uint8_t *> ring;
    std::vector<cudaEvent_t> ev_free, ev_ready;
    int ring_next = 0;
    cudaStream_t copy_stream = nullptr;

    uint64_t launches = 0;
    std::string last_error;

    // stream order of the ctx's shared scratch / aux / ring (StreamOrder): the end of the last
    // call is recorded on its stream; a call on another stream first waits on it
    cudaEvent_t ev_done = nullptr;
    cudaStream_t last_st = nullptr;
    bool last_valid = false;

    // hot-kernel profiling (shred_profile)
    bool prof = false;
    std::vector<cudaEvent_t> prof_ev;    // pool, pairs
    size_t prof_used = 0;
    uint64_t prof_bytes = 0;
};

namespace {

int fail(shred_ctx *c, int code, const char *fmt, ...) {
    if (c) {
        char buf[512];
        va_list ap; va_start(ap, fmt); vsnprintf(buf, sizeof buf, fmt, ap); va_end(ap);
        c->last_error = buf;
    }
    return code;
}
int cuda_fail(shred_ctx *c, cudaError_t e, const char *what) {
    return fail(c, SHRED_ECUDA, "%s: %s", what, cudaGetErrorString(e));
}
#define CK(call, what) do { cudaError_t _e = (call); if (_e != cudaSuccess) return cuda_fail(ctx, _e, what); } while (0)
#define LAUNCHED(what) do { ++ctx->launches; cudaError_t _e = cudaGetLastError(); if (_e != cudaSuccess) return cuda_fail(ctx, _e, what); } while (0)

// Programmatic dependent launch: every kernel of a call's chain is launched with programmatic
// stream serialization, and each starts with griddepcontrol.wait + launch_dependents
// (kernels.cuh pdl_entry), so a kernel's launch overlaps the tail of its predecessor instead of
// paying the full launch gap (small inputs are launch-latency-bound).
template <typename... KArgs, typename... Args>
cudaError_t pdl_launch(void (*k)(KArgs...), dim3 g, dim3 b, size_t smem, cudaStream_t st, Args... args) {
    cudaLaunchConfig_t cfg{};
    cfg.gridDim = g; cfg.blockDim = b; cfg.dynamicSmemBytes = smem; cfg.stream = st;
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[0].val.programmaticStreamSerializationAllowed = SHRED_PDL;
    cfg.attrs = at; cfg.numAttrs = 1;
    return cudaLaunchKernelEx(&cfg, k, static_cast<KArgs>(args)...);
}
#define PDL(k, g, b, smem, st, ...) do { cudaError_t _pe = pdl_launch(k, g, b, smem, st, __VA_ARGS__); \
    if (_pe != cudaSuccess) return cuda_fail(ctx, _pe, #k); } while (0)

// Scratch grows synchronously: freeing the old buffer waits for the whole device
// (cudaDeviceSynchronize), so a call that needs more scratch than any earlier call blocks the
// host once (include/shred.h "Streams").  Steady-state calls of the same or smaller size never do.
template <class T>
int grow(shred_ctx *ctx, T *&ptr, uint64_t &cap, uint64_t need, const char *what) {
    if (need <= cap) return SHRED_OK;
    uint64_t n = need + need / 4 + 64;
    if (ptr) { cudaDeviceSynchronize(); cudaFree(ptr); ptr = nullptr; cap = 0; }
    cudaError_t e = cudaMalloc(&ptr, n * sizeof(T));
    if (e != cudaSuccess) { cudaGetLastError(); return fail(ctx, SHRED_ENOMEM, "%s: cudaMalloc(%llu B) failed", what, (unsigned long long)(n * sizeof(T))); }
    cap = n;
    return SHRED_OK;
}

// MODE_K32T eligibility: deg P = k <= 32 and Q = P - x^k has its terms at least 8 apart and
// below k - 7, so t(x) Q(x) for a byte t is the integer product t * Q (the shifted copies of t
// never overlap) of degree < k (no second reduction).  The multiplier adds the cancel term:
// M = Q + 2^k mod 2^32.
// Degrees 41..63 (MODE_K63T): Q's terms at least 8 apart and below 25, so t(x) Q(x) = t * Q fits
// the low word; the cancel term (t << k) mod 2^64 is t * 2^(k-32) in the high word (mult_hi).
bool tprod_ok(uint64_t P, int k, uint32_t *mult, uint32_t *mult_hi = nullptr) {
    const bool u64 = k >= 41 && k <= 63;
    if (!u64 && (k < 9 || k > 32)) return false;
    const int top = u64 ? 32 : k;                  // every term e needs e + 7 < top
    const uint64_t Q = P ^ (1ull << k);
    int prev = -100;
    for (int e = 0; e < k; ++e) {
        if (!((Q >> e) & 1u)) continue;
        if (e - prev < 8 || e + 7 >= top) return false;
        prev = e;
    }
    if (mult) *mult = u64 ? (uint32_t)Q : (uint32_t)(Q + (k < 32 ? (1ull << k) : 0ull));
    if (mult_hi) *mult_hi = u64 ? (1u << (k - 32)) : 0u;
    return true;
}

// Validation of shred_params (include/shred.h).
int validate(const shred_params *p, shred_ctx *ctx) {
    if (!p) return fail(ctx, SHRED_EINVAL, "params is NULL");
    const int k = deg64(p->poly);
    if (k < 8 || k > 63) return fail(ctx, SHRED_EINVAL, "deg(poly) = %d, need 8..63", k);
    if (!irreducible(p->poly)) return fail(ctx, SHRED_EINVAL, "poly 0x%llx is reducible", (unsigned long long)p->poly);
    if (p->window < 1 || p->window > 4096) return fail(ctx, SHRED_EINVAL, "window %u not in 1..4096", p->window);
    if (p->marker > SHRED_MARKER_LE) return fail(ctx, SHRED_EINVAL, "marker must be SHRED_MARKER_EQ or SHRED_MARKER_LE");
    if (p->divisor < 2) return fail(ctx, SHRED_EINVAL, "divisor must be >= 2");
    if (p->divisor > (1ull << k)) return fail(ctx, SHRED_EINVAL, "divisor exceeds 2^deg(poly)");
    if (p->magic >= p->divisor) return fail(ctx, SHRED_EINVAL, "magic must be < divisor");
    if (p->max_size && p->max_size < (p->min_size > 1 ? p->min_size : 1))
        return fail(ctx, SHRED_EINVAL, "max_size must be >= max(min_size, 1)");
    return SHRED_OK;
}

// Kernel path and marker kind for valid parameters on an sm_100a device.  The hot kernel takes
// any w <= 64 (w % 16 != 0: funnel-shifted pops), and D = 2^m <= 2^32 with either marker set on
// the low word, the '==' marker with any D = d 2^s (s < 32) by the divisibility test on the
// full state (MK_DIV), and every other D by the remainder itself (MK_REM).  u64 state: deg 33..63 (top byte by mulhi, or a funnel shift for k <= 40);
// u32 state: deg 9..32, and 8 (its top byte is the whole state: the PRMT byte index of
// MODE_K32B).  Windows 65..LW_MAX: the same kernel with the pops from a second TMA tile (WCH = 0
// instances, "long windows"); longer ones: the generic loop.
constexpr uint32_t LW_MAX = 4096;   // longest window of the hot kernel (16 ceil(w/16) <= GS * NTC)
int select_path(const shred_params *p, int *mk) {
    const int k = deg64(p->poly);
    const bool pow2 = (p->divisor & (p->divisor - 1)) == 0;
    const bool fast_w = p->window >= 1 && p->window <= LW_MAX;
    if (pow2 && p->divisor <= (1ull << 32)) *mk = p->marker == SHRED_MARKER_LE ? MK_LE : MK_EQ;
    else if (p->marker == SHRED_MARKER_EQ && __builtin_ctzll(p->divisor) < 32) *mk = MK_DIV;
    else *mk = MK_REM;
    const bool fast = fast_w && *mk >= 0;
    if (k >= 33 && k <= 63 && fast) return SHRED_PATH_K63;
    if ((k >= 9 || (k == 8 && SHRED_BYTEIDX)) && k <= 32 && fast) return SHRED_PATH_K32;
    return SHRED_PATH_GENERIC;
}

// ---------------------------------------------------------------------------- job planning
struct Plan {
    Job J;
    bool bulk = false;
    bool small = false;                  // bulk with the CfgSmall launch shape
    uint32_t nslots = 0;
    uint32_t bulk_ctas = 0;
    CUtensorMap tmap;
    CUtensorMap tmap_pop;                // long windows: the pop tiles (16 ceil(w/16) bytes behind)
};

// The pure part of planning (no device state; shred_debug_plan exposes it to CPU tests): the
// slot map of window ends [t_begin, t_end) of a job whose bytes start at stream position p_begin
// at address src_addr.  Fast paths: an aligned bulk region [b0, b0 + nrows*S) of rows for
// k1_bulk, head segments [t_begin, b0) and tail segments for its edge CTA (at most NTC each:
// one thread per segment).  Otherwise generic segments only.  Returns the row length S.
// warm: bytes each row rolls before its first window end (16 * ceil(w / 16)); zero_lead: the
// job starts at the stream start with no carried prefix (virtual zero bytes before it).
struct MapShape { bool fast; bool k63; bool small_ok; int sm_count; uint32_t warm; bool zero_lead; };
uint64_t plan_map(const MapShape &sh, uint64_t src_addr, uint64_t p_begin, uint64_t t_begin,
                  uint64_t t_end, SlotMap &m, bool &bulk, bool &small) {
    m = SlotMap{};
    m.t_end = t_end;
    const uint64_t len = t_end > t_begin ? t_end - t_begin : 0;
    const uint64_t GS = SHRED_EDGE_GS;         // head/tail segment (edge CTA)
    uint64_t ROWS_CTA = sh.k63 ? CfgK63::ROWS : CfgK32::ROWS;
    uint64_t NTC = sh.k63 ? CfgK63::NTC : CfgK32::NTC;
    bulk = false;
    small = false;
    uint64_t S = 0, nrows = 0, b0 = t_end;
    if (sh.fast && len >= 4096) {
        // bulk region: aligned start b0 >= max(t_begin, p_begin + warm), rows of S bytes; at the
        // start of a stream with no carry the first row may start at the stream start itself
        // (its warm-up reads virtual zero bytes), so an aligned stream needs no head segments
        uint64_t lo = t_begin > p_begin + sh.warm ? t_begin : p_begin + sh.warm;
        if (sh.zero_lead && t_begin == p_begin && (src_addr & 15u) == 0) lo = p_begin;
        const uint64_t a = src_addr + (lo - p_begin);
        b0 = lo + ((16u - (a & 15u)) & 15u);
        if (b0 + 256 < t_end) {
            const uint64_t blen = t_end - b0;
            // one wave: (SMs - 1) bulk CTAs of ROWS_CTA rows + the edge CTA
            const uint64_t sms = (uint64_t)(sh.sm_count > 1 ? sh.sm_count - 1 : 1);
            uint64_t target = sms * ROWS_CTA;
            if (sh.small_ok && blen <= target * 32) {
                // rows of < 64 B with the big shape: use the small one, two CTAs per SM
                // (tools/size_latency.py: faster up to ~4 MiB, slower from ~16 MiB)
                small = true;
                ROWS_CTA = CfgSmall::ROWS; NTC = CfgSmall::NTC;
                target = 2 * sms * ROWS_CTA;
            }
            S = (blen + target - 1) / target;
            S = (S + 31) / 32 * 32;                // whole 32-byte rounds (16-byte rounds for CH = 4)
            if (S < 32) S = 32;                    // small inputs: short rows, each a chain of w + S steps
            nrows = blen / S;
            if (nrows > 0 && nrows < (1ull << 31) && S < (1ull << 39) && (b0 - t_begin) <= GS * NTC)
                bulk = true;
        }
    }
    if (!bulk) {
        small = false;
        // generic only: segments of about len / (sm_count * 4 * 256) bytes, >= 256
        uint64_t seg = 256;
        const uint64_t want = (uint64_t)sh.sm_count * 4 * GEN_THREADS;
        if (len / want > seg) seg = (len / want + 63) / 64 * 64;
        m.head_start = t_begin; m.head_seg = seg;
        m.n_head = (uint32_t)((len + seg - 1) / seg);
        m.nrows = 0; m.b0 = t_end; m.S = 0;
        m.tail_start = t_end; m.tail_seg = seg; m.n_tail = 0;
        m.nc = 0;
        m.ngroups = (m.n_head + GEN_THREADS - 1) / GEN_THREADS;
        return 0;
    }
    m.head_start = t_begin; m.head_seg = GS;
    m.n_head = (uint32_t)((b0 - t_begin + GS - 1) / GS);
    m.b0 = b0; m.S = S; m.nrows = (uint32_t)nrows;
    m.tail_start = b0 + nrows * S;
    const uint64_t tl = t_end - m.tail_start;
    uint64_t ts = (tl + NTC - 1) / NTC;
    ts = ts < GS ? GS : (ts + 15) / 16 * 16;
    m.tail_seg = ts;
    m.n_tail = (uint32_t)((tl + ts - 1) / ts);
    m.nc = (uint32_t)((nrows + ROWS_CTA - 1) / ROWS_CTA);
    m.rows_cta = (uint32_t)ROWS_CTA;
    m.ngroups = m.nc + 2;
    return S;
}

// Per-slot list capacity: twice the expected count of the longest segment + slack.  The hit
// rate is 1/D for the '==' marker and (r+1)/D for the '<=' set (sizing '<=' lists
// by 1/D overflowed every list for a large r, sending unbounded calls to the re-roll and
// bounded calls to the one-CTA sb_dense walk).  At most SLOT_CAP_MAX entries per slot, and the
// lists of all slots stay within SCRATCH_BUDGET bytes; beyond that the input is dense and the
// overflow paths (exact) take over.
constexpr uint64_t SLOT_CAP_MAX = 4096;
constexpr uint64_t SCRATCH_BUDGET = 4ull << 30;
uint32_t slot_cap(const SlotMap &m, bool bulk, uint64_t divisor, uint64_t hits_per_d, uint64_t nslots) {
    uint64_t maxseg = bulk ? m.S : m.head_seg;
    if (bulk && m.tail_seg > maxseg) maxseg = m.tail_seg;
    const long double exp = (long double)maxseg * (long double)hits_per_d / (long double)divisor;
    long double capf = 2.0L * exp + 16.0L;
    if (capf > (long double)SLOT_CAP_MAX) capf = (long double)SLOT_CAP_MAX;
    uint64_t cap = (uint64_t)capf;
    if (nslots && cap * 8 * nslots > SCRATCH_BUDGET) cap = SCRATCH_BUDGET / 8 / nslots;
    if (cap < 16) cap = 16;
    return (uint32_t)cap;
}
// candidate hits per D positions for the ctx's marker set: 1 ('=='), r + 1 ('<=')
uint64_t hits_per_d(const shred_params &p) { return p.marker == SHRED_MARKER_LE ? p.magic + 1 : 1; }

// Plan candidate detection for window ends [t_begin, t_end) of a job whose bytes start at
// stream position p_begin (src) with `prefix_len` carried bytes before it.
int plan_job(shred_ctx *ctx, Plan &pl, const uint8_t *src, uint64_t p_begin, const uint8_t *prefix,
             uint32_t prefix_len, uint64_t t_begin, uint64_t t_end, uint64_t c_limit) {
    Job &J = pl.J;
    J = Job{};
    J.src = src; J.p_begin = p_begin; J.prefix = prefix; J.prefix_len = prefix_len;
    J.min_i = (uint64_t)ctx->p.window - 1u;
    J.c_limit = c_limit;
    SlotMap &m = J.map;
    const MapShape sh{ctx->path == SHRED_PATH_K63 || ctx->path == SHRED_PATH_K32, ctx->path == SHRED_PATH_K63,
                      ctx->k1_small_fn != nullptr, ctx->sm_count, 16u * ((ctx->p.window + 15u) / 16u),
                      prefix_len == 0 && ctx->p.window <= 64};   // long windows: pop tiles stay inside src
    const uint64_t S = plan_map(sh, (uint64_t)(uintptr_t)src, p_begin, t_begin, t_end, m, pl.bulk, pl.small);
    if (pl.bulk) {
        const uint64_t ROUND = CfgK63::ROUND;
        static_assert(CfgK63::ROUND == CfgSmall::ROUND && CfgK32::ROUND == CfgSmall::ROUND, "round");
        pl.bulk_ctas = m.nc + 1;               // + the edge CTA (head + tail, group sums 0, nc+1)
        // 2-D tensor map [nrows][S] over the bulk bytes
        cuuint64_t gdim[2] = {(cuuint64_t)S, (cuuint64_t)m.nrows};
        cuuint64_t gstride[1] = {(cuuint64_t)S};
        cuuint32_t box[2] = {(cuuint32_t)ROUND, (cuuint32_t)(pl.small ? CfgSmall::BOX : CfgK63::BOX)};
        static_assert(CfgK63::BOX == CfgK32::BOX, "box");
        cuuint32_t estr[2] = {1, 1};
        // the same buffer chunked again (a loop over one buffer, configs[0]-size calls) reuses the
        // last encoded map: the host cost of a small call is part of its latency
        const uint64_t key[4] = {(uint64_t)(uintptr_t)(src + (m.b0 - p_begin)), S, (uint64_t)m.nrows, box[1]};
        if (ctx->tm_valid && memcmp(key, ctx->tm_key, sizeof key) == 0) {
            pl.tmap = ctx->tm_cache;
        } else {
            CUresult r = ctx->encode(&pl.tmap, CU_TENSOR_MAP_DATA_TYPE_UINT8, 2,
                                     (void *)(src + (m.b0 - p_begin)), gdim, gstride, box, estr,
                                     CU_TENSOR_MAP_INTERLEAVE_NONE,
                                     ROUND == 64 ? CU_TENSOR_MAP_SWIZZLE_64B
                                                 : (ROUND == 32 ? CU_TENSOR_MAP_SWIZZLE_32B : CU_TENSOR_MAP_SWIZZLE_NONE),
                                     (CUtensorMapL2promotion)SHRED_L2PROMO, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
            if (r != CUDA_SUCCESS) return fail(ctx, SHRED_ECUDA, "cuTensorMapEncodeTiled failed (%d)", (int)r);
            ctx->tm_cache = pl.tmap;
            memcpy(ctx->tm_key, key, sizeof key);
            ctx->tm_valid = true;
        }
        if (ctx->p.window > 64) {
            // long windows: rows of the same geometry 16 ceil(w/16) bytes earlier (the plan keeps
            // b0 - 16 ceil(w/16) >= p_begin), 48-byte boxes (two pop chunks + the funnel's next)
            const uint64_t back = 16ull * ((ctx->p.window + 15u) / 16u);
            cuuint32_t pbox[2] = {(cuuint32_t)LW_POPW, box[1]};
            CUresult r = ctx->encode(&pl.tmap_pop, CU_TENSOR_MAP_DATA_TYPE_UINT8, 2,
                                     (void *)(src + (m.b0 - back - p_begin)), gdim, gstride, pbox, estr,
                                     CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE,
                                     (CUtensorMapL2promotion)SHRED_L2PROMO, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
            if (r != CUDA_SUCCESS) return fail(ctx, SHRED_ECUDA, "cuTensorMapEncodeTiled (pops) failed (%d)", (int)r);
        }
    }
    pl.nslots = m.n_head + m.nrows + m.n_tail;
    if (m.ngroups > (uint32_t)MAX_GROUPS) return fail(ctx, SHRED_EINVAL, "too many slot groups (%u)", m.ngroups);
    pl.nslots = m.n_head + m.nrows + m.n_tail;
    J.cap = slot_cap(m, pl.bulk, ctx->p.divisor, hits_per_d(ctx->p), pl.nslots);
    int rc;
    if ((rc = grow(ctx, ctx->d_counts, ctx->counts_cap, (uint64_t)pl.nslots + 1, "counts"))) return rc;
    if ((rc = grow(ctx, ctx->d_local, ctx->local_cap, (uint64_t)pl.nslots + 1, "local offsets"))) return rc;
    if ((rc = grow(ctx, ctx->d_groups, ctx->groups_cap, (uint64_t)m.ngroups + 1, "group sums"))) return rc;
    if ((rc = grow(ctx, ctx->d_scratch, ctx->scratch_cap, (uint64_t)pl.nslots * J.cap + 1, "scratch"))) return rc;
    J.counts = ctx->d_counts;
    J.local_off = ctx->d_local;
    J.group_sum = ctx->d_groups;
    J.scratch = ctx->d_scratch;
    return SHRED_OK;
}

// K1: the TMA hot kernel (+ its edge CTA), or the generic kernel.
int launch_detect(shred_ctx *ctx, Plan &pl, cudaStream_t st) {
    if (pl.nslots == 0) return SHRED_OK;
    if (pl.bulk) {
        cudaEvent_t e0 = nullptr, e1 = nullptr;
        if (ctx->prof) {
            if (ctx->prof_used + 2 > ctx->prof_ev.size()) {
                for (int i = 0; i < 64; ++i) {
                    cudaEvent_t e;
                    CK(cudaEventCreate(&e), "profile event");
                    ctx->prof_ev.push_back(e);
                }
            }
            e0 = ctx->prof_ev[ctx->prof_used]; e1 = ctx->prof_ev[ctx->prof_used + 1];
            ctx->prof_used += 2;
            ctx->prof_bytes += (pl.J.map.t_end - pl.J.map.head_start);
            CK(cudaEventRecord(e0, st), "profile record");
        }
        const int m = ctx->mk >= MK_DIV ? 0 : 32 - (int)__builtin_ctzll(ctx->p.divisor);   // D = 2^(32-m)
        BulkConst K;
        // top byte t = f >> (k-8): u64 state mulhi(f_hi, 2^(72-k)); u32 state mulhi(f, 2^(40-k))
        K.mhi = ctx->path == SHRED_PATH_K63 ? (ctx->k >= 41 ? (1u << (72 - ctx->k)) : (uint32_t)(ctx->k - 8))
                                            : (ctx->k >= 9 ? (1u << (40 - ctx->k)) : 0u);   // deg 8: byte index
        const uint32_t e = (uint32_t)(16 * ((ctx->p.window + 15) / 16) - ctx->p.window);
        K.fu = e / 4;
        K.wa = (uint32_t)((ctx->p.window + 15) / 16);
        K.fsel = 0x3210u + 0x1111u * (e % 4);
        K.m256 = 256u;
        K.tmul = 1u << m;                                           // 2^(32 - log2 D)
        K.rsh = (uint32_t)(ctx->p.magic << m);
        K.tshr = (uint32_t)(ctx->k >= 41 ? ctx->k - 40 : ctx->k - 8);
        K.tprod = 0u; K.tprod_hi = 0u;
        K.dm32 = (uint32_t)(ctx->p.divisor - 1u); K.r32 = (uint32_t)ctx->p.magic;
        tprod_ok(ctx->p.poly, ctx->k, &K.tprod, &K.tprod_hi);
        {   // MK_DIV: D = d 2^s; d^-1 mod 2^64 by Newton's iteration (d odd: d*d = 1 mod 8)
            const uint64_t D = ctx->p.divisor;
            const uint32_t sh = (uint32_t)__builtin_ctzll(D);
            const uint64_t d = D >> sh;
            uint64_t inv = d;
            for (int it = 0; it < 5; ++it) inv *= 2u - d * inv;
            K.dc = D - ctx->p.magic; K.dinv = inv; K.dlim = ~0ull / D; K.dsh = sh;
            // MK_REM: l = ceil(log2 D) in 1..63; rm = ceil(2^(63+l) / D) < 2^64 (D > 2^(l-1), or
            // D = 2^l and rm = 2^63); q = mulhi(f, rm) >> (l-1) = floor(f / D) for every f < 2^63
            const int l = 64 - __builtin_clzll(D - 1);
            const unsigned __int128 num = (unsigned __int128)1 << (63 + l);
            K.rm = (uint64_t)((num + D - 1) / D); K.rd = D; K.rsh2 = (uint32_t)(l - 1);
            K.rlo = ctx->p.marker == SHRED_MARKER_LE ? 0 : ctx->p.magic;
            K.rspan = ctx->p.marker == SHRED_MARKER_LE ? ctx->p.magic : 0;
        }
        K.tsel = 0x5504u | ((uint32_t)((ctx->k - 8) / 8) << 4);         // byte (k-8)/8 -> bits 8..15
        K.pos = ctx->d_pos; K.w = ctx->p.window;
        int smem = ctx->k1_smem;
        int threads = (ctx->path == SHRED_PATH_K63 ? CfgK63::NTC : CfgK32::NTC) + 32;
        K1Fn fn = ctx->k1_fn;
        if (pl.small) { smem = CfgSmall::SMEM; threads = CfgSmall::NTC + 32; fn = ctx->k1_small_fn; }
        PDL(fn, pl.bulk_ctas, threads, smem, st, pl.tmap, ctx->p.window > 64 ? pl.tmap_pop : pl.tmap,
            ctx->d_tab_img, ctx->d_gen, pl.J, ctx->dp, K);
        LAUNCHED("k1_bulk");
        if (e1) CK(cudaEventRecord(e1, st), "profile record");
    } else {
        PDL(k1_generic, (pl.nslots + GEN_THREADS - 1) / GEN_THREADS, GEN_THREADS, 0, st, pl.J, ctx->dp, ctx->d_gen,
                                                                                       pl.nslots);
        LAUNCHED("k1_generic");
    }
    return SHRED_OK;
}

// Ordered compaction into dst.  With no slots: total = 0 (and *n_direct = 0).
int launch_scatter(shred_ctx *ctx, Plan &pl, uint64_t *dst, uint64_t dst_cap, Aux *aux, int streaming,
                   uint64_t *n_direct, cudaStream_t st, int reset = 0) {
    if (pl.nslots == 0) {
        PDL(k_no_slots, 1, 1, 0, st, aux, n_direct, reset);
        LAUNCHED("k_no_slots");
        return SHRED_OK;
    }
    PDL(k_scatter, (pl.nslots + SCATTER_THREADS - 1) / SCATTER_THREADS, SCATTER_THREADS, 0, st, 
        pl.J, ctx->dp, ctx->d_gen, pl.nslots, dst, dst_cap, aux, streaming, n_direct, reset);
    LAUNCHED("k_scatter");
    return SHRED_OK;
}

bool bounded(const shred_ctx *ctx) { return ctx->p.min_size > 0 || ctx->p.max_size > 0; }

// The size rule over ascending candidates.  `nmax` bounds the count for the grid sizes; the
// kernels read the true count from n_dev if given (else n_host).  Appends to dst at
// aux->out_pos; updates aux.  With `pl` given, the dense fallback (sb_dense) is enqueued too: it
// runs only if the ordered list could not hold every candidate.
int launch_size_bound(shred_ctx *ctx, const uint64_t *cand, const uint64_t *n_dev, uint64_t n_host,
                      uint64_t nmax, uint64_t end, int fin, uint64_t *dst, uint64_t cap, Aux *aux,
                      const Plan *pl, cudaStream_t st, uint64_t *n_out = nullptr) {
    // blocks of 8 candidates when min <= half the mean candidate gap (D / h), else 16 (size_bound.cuh)
    const bool small_b = (long double)ctx->p.min_size * 2.0L * (long double)hits_per_d(ctx->p) <=
                         (long double)ctx->p.divisor;
    const int B = small_b ? SB_B_SMALL : SB_B;
    const uint64_t nb = (nmax + B - 1) / B;
    int rc = grow(ctx, ctx->d_sb, ctx->sb_cap, 9 * (nb + 2), "size-rule scratch");
    if (rc) return rc;
    SBArgs A;
    A.cand = cand; A.n_dev = n_dev; A.n_host = n_host; A.n_cap = nmax;
    A.minsz = ctx->p.min_size; A.maxsz = ctx->p.max_size; A.end = end; A.fin = fin;
    uint64_t *b = ctx->d_sb;
    A.spec_exit = b; A.spec_cnt = b + (nb + 2); A.entry = b + 2 * (nb + 2); A.offs = b + 3 * (nb + 2);
    A.delta = (int64_t *)(b + 4 * (nb + 2)); A.ok = (uint32_t *)(b + 5 * (nb + 2));
    A.cta_sum = b + 6 * (nb + 2); A.cta_ok = b + 7 * (nb + 2); A.cta_off = b + 8 * (nb + 2);
    A.dst = dst; A.dst_cap = cap; A.aux = aux; A.tile = SB_THREADS; A.n_out = n_out;
    // tiles of SB_THREADS blocks, at most 8 CTAs per SM (grid-stride over the true tile count)
    const uint64_t gmax = (uint64_t)ctx->sm_count * 8;
    uint64_t g = (nb + SB_THREADS - 1) / SB_THREADS;
    if (g > gmax) g = gmax;
    if (nb) {
        if (small_b) { PDL(sb_spec_check<SB_B_SMALL>, (unsigned)g, SB_THREADS, 0, st, A); }
        else         { PDL(sb_spec_check<SB_B>, (unsigned)g, SB_THREADS, 0, st, A); }
        LAUNCHED("sb_spec_check");
    }
    if (small_b) { PDL(sb_plan<SB_B_SMALL>, 1, 1024, 0, st, A); }
    else         { PDL(sb_plan<SB_B>, 1, 1024, 0, st, A); }
    LAUNCHED("sb_plan");
    uint64_t ge = (nb + 1 + SB_THREADS - 1) / SB_THREADS;
    if (ge > gmax) ge = gmax;
    if (small_b) { PDL(sb_emit<SB_B_SMALL>, (unsigned)ge, SB_THREADS, 0, st, A); }
    else         { PDL(sb_emit<SB_B>, (unsigned)ge, SB_THREADS, 0, st, A); }
    LAUNCHED("sb_emit");
    if (pl && pl->nslots) {
        uint64_t maxseg = pl->J.map.S;
        if (pl->J.map.head_seg > maxseg) maxseg = pl->J.map.head_seg;
        if (pl->J.map.tail_seg > maxseg) maxseg = pl->J.map.tail_seg;
        if (maxseg > SBD_WIN) maxseg = SBD_WIN;
        const size_t smem = (size_t)((maxseg + 31) / 32) * 4;
        PDL(sb_dense, 1, SBD_THREADS, smem, st, pl->J, ctx->dp, ctx->d_gen, pl->nslots, A);
        LAUNCHED("sb_dense");
    }
    return SHRED_OK;
}

// One piece of a stream (or a whole one-shot stream): window ends [t_begin, t_end).
// aux->out_pos is the output cursor; results are appended to dst.
int run_piece(shred_ctx *ctx, Aux *aux, const uint8_t *src, uint64_t p_begin, const uint8_t *prefix,
              uint32_t prefix_len, uint64_t t_begin, uint64_t t_end, uint64_t c_limit, int final_,
              uint64_t *dst, uint64_t dst_cap, cudaStream_t st) {
    Plan pl;
    int rc = plan_job(ctx, pl, src, p_begin, prefix, prefix_len, t_begin, t_end, c_limit);
    if (rc) return rc;
    if ((rc = launch_detect(ctx, pl, st))) return rc;
    if (!bounded(ctx)) {
        if ((rc = launch_scatter(ctx, pl, dst, dst_cap, aux, 1, nullptr, st))) return rc;
        if (final_) {
            // one-shot: nothing held; out_pos += total
            PDL(k_piece_done, 1, 1, 0, st, aux, dst, dst_cap, ~0ull);
        } else {
            PDL(k_piece_done, 1, 1, 0, st, aux, dst, dst_cap, t_end);
        }
        LAUNCHED("k_piece_done");
        return SHRED_OK;
    }
    // ordered candidate list: every slot's complete list fits (dense inputs -> sb_dense)
    const uint64_t ccap = (uint64_t)pl.nslots * pl.J.cap + 1;
    if ((rc = grow(ctx, ctx->d_cand, ctx->cand_cap, ccap, "candidate list"))) return rc;
    if ((rc = launch_scatter(ctx, pl, ctx->d_cand, ccap, aux, 0, nullptr, st))) return rc;
    return launch_size_bound(ctx, ctx->d_cand, &aux->ncand, 0, ccap, t_end, final_, dst, dst_cap, aux,
                             &pl, st);
}

// Kind of a user pointer: 1 = device, 2 = page-locked host, 0 = pageable / unknown.
int ptr_kind(const void *p) {
    cudaPointerAttributes a;
    cudaError_t e = cudaPointerGetAttributes(&a, p);
    if (e != cudaSuccess) { cudaGetLastError(); return 0; }
    if (a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged) return 1;
    if (a.type == cudaMemoryTypeHost) return 2;
    return 0;
}

int check_out(shred_ctx *ctx, uint64_t *d_out, uint64_t cap, uint64_t *n_out) {
    if (!n_out) return fail(ctx, SHRED_EINVAL, "n_out is NULL");
    if (cap && !d_out) return fail(ctx, SHRED_EINVAL, "d_out is NULL with cap > 0");
    return SHRED_OK;
}

struct DevGuard {
    int prev = -1;
    explicit DevGuard(int dev) { cudaGetDevice(&prev); if (prev != dev) cudaSetDevice(dev); }
    ~DevGuard() { if (prev >= 0) cudaSetDevice(prev); }
};

// Every call's work uses the ctx's scratch, aux state and ring, so calls on one ctx must run in
// order even when they are enqueued on different streams (two one-shot calls on two
// streams raced on d_aux[0] and the scratch lists).  The guard makes a call on a stream other
// than the previous call's wait for that call's completion event, and records its own at the
// end.  Under stream capture (CUDA graphs) nothing is recorded or waited on: a captured call
// must be captured on the stream the ctx's preceding work used (include/shred.h "Streams").
// The event is recorded lazily: only when a call arrives on a different stream is the end of the
// previous stream's work (everything enqueued on it so far, which includes the previous call)
// recorded there and waited on; consecutive calls on one stream cost no event (host time of a
// small call matters: configs[0]).
struct StreamOrder {
    StreamOrder(shred_ctx *ctx, cudaStream_t st) {
        if (ctx->last_valid && ctx->last_st == st) return;
        cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone, cp = cudaStreamCaptureStatusNone;
        if (cudaStreamIsCapturing(st, &cs) != cudaSuccess) cudaGetLastError();
        if (ctx->last_valid && cudaStreamIsCapturing(ctx->last_st, &cp) != cudaSuccess) cudaGetLastError();
        if (ctx->last_valid && cs == cudaStreamCaptureStatusNone && cp == cudaStreamCaptureStatusNone) {
            if (cudaEventRecord(ctx->ev_done, ctx->last_st) == cudaSuccess) cudaStreamWaitEvent(st, ctx->ev_done, 0);
            else cudaGetLastError();
        }
        ctx->last_st = st;
        ctx->last_valid = cs == cudaStreamCaptureStatusNone;
    }
};

}  // namespace

// ============================================================================ C ABI
extern "C" {

void shred_default_params(shred_params *p) {
    if (!p) return;
    memset(p, 0, sizeof *p);
    p->poly = 0xbfe6b8a5bf378d83ull;
    p->window = 48;
    p->divisor = 8192;
    p->magic = 0x78;
}

const char *shred_strerror(int code) {
    if (code > 0 || code < -5) return "unknown error";
    return kErr[-code];
}

const char *shred_last_error(const shred_ctx *ctx) { return ctx ? ctx->last_error.c_str() : "no ctx"; }
int shred_path(const shred_ctx *ctx) { return ctx ? ctx->path : 0; }
int shred_kernel_mode(const shred_ctx *ctx) { return ctx ? ctx->mode : 0; }
uint64_t shred_launch_count(const shred_ctx *ctx) { return ctx ? ctx->launches : 0; }

int shred_get_params(const shred_ctx *ctx, shred_params *out) {
    if (!ctx || !out) return SHRED_EINVAL;
    *out = ctx->p;
    return SHRED_OK;
}

uint64_t shred_max_cuts(const shred_ctx *ctx, uint64_t len) {
    if (!ctx || len < 2) return 0;
    if (ctx->p.min_size == 0) return len - 1;
    return (len - 1) / ctx->p.min_size + 1;
}

int shred_init(const shred_params *p, int device, shred_ctx **out) {
    if (!out) return SHRED_EINVAL;
    *out = nullptr;
    int rc = validate(p, nullptr);
    if (rc) return rc;
    shred_ctx *ctx = new shred_ctx();
    ctx->p = *p;
    ctx->device = device;
    DevGuard g(device);
    auto bail = [&](int code) { shred_destroy(ctx); return code; };
    cudaError_t e = cudaSetDevice(device);
    if (e != cudaSuccess) return bail(SHRED_ECUDA);
    int major = 0;
    cudaDeviceGetAttribute(&major, cudaDevAttrComputeCapabilityMajor, device);
    cudaDeviceGetAttribute(&ctx->sm_count, cudaDevAttrMultiProcessorCount, device);
    if (ctx->sm_count <= 0) ctx->sm_count = 148;

    const int k = deg64(p->poly);
    ctx->k = k;
    ctx->dp.k = (uint32_t)k;
    ctx->dp.w = p->window;
    ctx->dp.kmask = (1ull << k) - 1ull;
    ctx->dp.dmask = p->divisor - 1ull;
    ctx->dp.magic = p->magic;
    ctx->dp.divisor = p->divisor;
    ctx->dp.pow2 = (p->divisor & (p->divisor - 1)) == 0 ? 1u : 0u;
    ctx->dp.marker = p->marker;
    ctx->path = select_path(p, &ctx->mk);
    if (major != 10) ctx->path = SHRED_PATH_GENERIC;   // the TMA kernels are built for sm_100a only

    // ---- tables (PAPER.md: shift one byte in, one byte out)
    uint64_t Tk[256], U[256];
    byte_times_xpow(p->poly, k, (uint64_t)k, Tk);                 // t x^k mod P
    byte_times_xpow(p->poly, k, 8ull * p->window, U);             // o x^{8w} mod P
    GenTables gt;
    for (int t = 0; t < 256; ++t) { gt.T[t] = Tk[t]; gt.U[t] = U[t]; }
    std::vector<uint8_t> img(TAB_BYTES, 0);
    // Fast-path T entries carry the cancel term (t << k) mod 2^W: after (f << 8) mod 2^W the top
    // byte t of f sits at bits k..k+7 (those below W); T[t] removes it and adds t x^k mod P.
    if (ctx->path == SHRED_PATH_K63) {
        for (int t = 0; t < 256; ++t) {
            uint64_t tv = Tk[t] ^ ((uint64_t)t << k);             // W = 64 (k = 63: (t&1) << 63)
            for (int r = 0; r < 16; ++r) {
                memcpy(&img[t * 256 + r * 8], &tv, 8);
                memcpy(&img[t * 256 + 128 + r * 8], &U[t], 8);
            }
        }
    } else if (ctx->path == SHRED_PATH_K32) {
        for (int t = 0; t < 256; ++t) {
            uint32_t tv = (uint32_t)(Tk[t] ^ ((uint64_t)t << k)), uv = (uint32_t)U[t];   // W = 32
            for (int r = 0; r < 32; ++r) {
                memcpy(&img[t * 256 + r * 4], &tv, 4);
                memcpy(&img[t * 256 + 128 + r * 4], &uv, 4);
            }
        }
    }
    if (cudaMalloc(&ctx->d_gen, sizeof(GenTables)) != cudaSuccess ||
        cudaMalloc(&ctx->d_tab_img, TAB_BYTES) != cudaSuccess ||
        cudaMalloc(&ctx->d_aux, 2 * sizeof(Aux)) != cudaSuccess ||
        cudaMalloc(&ctx->d_carry[0], 4096) != cudaSuccess ||
        cudaMalloc(&ctx->d_carry[1], 4096) != cudaSuccess ||
        cudaMalloc(&ctx->d_queue, 64) != cudaSuccess ||
        cudaMalloc(&ctx->d_hhist, HB * sizeof(uint32_t)) != cudaSuccess ||
        cudaHostAlloc(&ctx->h_pinned, 64, cudaHostAllocDefault) != cudaSuccess ||
        cudaHostAlloc(&ctx->h_flag, 64, cudaHostAllocMapped) != cudaSuccess ||
        cudaHostGetDevicePointer((void **)&ctx->d_flag, ctx->h_flag, 0) != cudaSuccess) {
        cudaGetLastError();
        return bail(SHRED_ENOMEM);
    }
    ctx->h_flag[0] = 0;
    if (cudaMemcpy(ctx->d_gen, &gt, sizeof gt, cudaMemcpyHostToDevice) != cudaSuccess ||
        cudaMemcpy(ctx->d_tab_img, img.data(), TAB_BYTES, cudaMemcpyHostToDevice) != cudaSuccess ||
        cudaMemset(ctx->d_aux, 0, 2 * sizeof(Aux)) != cudaSuccess)
        return bail(SHRED_ECUDA);
    if (ctx->path != SHRED_PATH_GENERIC) {
        void *fn = nullptr;
        cudaDriverEntryPointQueryResult q;
        if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fn, cudaEnableDefault, &q) != cudaSuccess || !fn)
            return bail(SHRED_ECUDA);
        ctx->encode = (EncodeTiledFn)fn;
        const bool byteidx = SHRED_BYTEIDX && ctx->path == SHRED_PATH_K32 && (k == 8 || k == 16 || k == 24 || k == 32);
        const int wch = p->window <= 64 ? (int)((p->window + 15) / 16) : 0;   // 0: long window
        const bool funnel = p->window % 16 != 0;
        const bool tprod = SHRED_TPROD && (ctx->path == SHRED_PATH_K32 || k >= 41) && tprod_ok(p->poly, k, nullptr);
        ctx->k1_fn = pick_k1(k, byteidx, wch, ctx->mk, funnel, tprod);
        const bool tmode = tprod && (ctx->mk == MK_EQ || ctx->mk == MK_LE);
        ctx->mode = ctx->path == SHRED_PATH_K63 ? (k >= 41 ? (tmode ? MODE_K63T : MODE_K63) : MODE_K40)
                  : tmode ? MODE_K32T : (byteidx ? MODE_K32B : MODE_K32);
        ctx->k1_smem = ctx->path == SHRED_PATH_K63 ? (wch ? CfgK63::SMEM : LwLayout<CfgK63>::SMEM)
                                                   : (wch ? CfgK32::SMEM : LwLayout<CfgK32>::SMEM);
        if (!ctx->k1_fn ||
            cudaFuncSetAttribute(ctx->k1_fn, cudaFuncAttributeMaxDynamicSharedMemorySize, ctx->k1_smem) != cudaSuccess)
            return bail(SHRED_ECUDA);
#ifdef SHRED_CARVEOUT   // A/B only: force the L1/SMEM split of the hot kernel (percent of max smem)
        cudaFuncSetAttribute(ctx->k1_fn, cudaFuncAttributePreferredSharedMemoryCarveout, SHRED_CARVEOUT);
#endif
#ifndef SHRED_NO_SMALL
        ctx->k1_small_fn = pick_k1_small(k, byteidx, wch, ctx->mk, funnel, tprod);
#endif
        if (ctx->k1_small_fn &&
            cudaFuncSetAttribute(ctx->k1_small_fn, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                 CfgSmall::SMEM) != cudaSuccess)
            return bail(SHRED_ECUDA);
        if (ctx->k1_small_fn && CfgSmall::DIRECT_WARM) {
            // the small shape's row start states: C_j[b] = b x^{8j} mod P (direct definition of
            // the window fingerprint), j < w <= 64: w x 2 KiB
            std::vector<uint64_t> pos(256 * (size_t)p->window);
            for (uint32_t j = 0; j < p->window; ++j) byte_times_xpow(p->poly, k, 8ull * j, &pos[256 * (size_t)j]);
            if (cudaMalloc(&ctx->d_pos, pos.size() * 8) != cudaSuccess) { cudaGetLastError(); return bail(SHRED_ENOMEM); }
            if (cudaMemcpy(ctx->d_pos, pos.data(), pos.size() * 8, cudaMemcpyHostToDevice) != cudaSuccess)
                return bail(SHRED_ECUDA);
        }
    }
    if (cudaFuncSetAttribute(sb_dense, cudaFuncAttributeMaxDynamicSharedMemorySize,
                             (int)(SBD_WIN / 8)) != cudaSuccess ||
        cudaFuncSetAttribute(sb_one, cudaFuncAttributeMaxDynamicSharedMemorySize,
                             (int)(SBD_WIN / 8 > SBO_SMEM ? SBD_WIN / 8 : SBO_SMEM)) != cudaSuccess ||
        cudaFuncSetAttribute(k_hash_chunks_ws, cudaFuncAttributeMaxDynamicSharedMemorySize,
                             (int)HWS_SMEM) != cudaSuccess)
        return bail(SHRED_ECUDA);
    if (cudaStreamCreateWithFlags(&ctx->copy_stream, cudaStreamNonBlocking) != cudaSuccess ||
        cudaEventCreateWithFlags(&ctx->ev_done, cudaEventDisableTiming) != cudaSuccess)
        return bail(SHRED_ECUDA);
    if (cudaDeviceSynchronize() != cudaSuccess) return bail(SHRED_ECUDA);
    *out = ctx;
    return SHRED_OK;
}

void shred_destroy(shred_ctx *ctx) {
    if (!ctx) return;
    DevGuard g(ctx->device);
    if (ctx->copy_stream) cudaStreamSynchronize(ctx->copy_stream);
    cudaDeviceSynchronize();
    for (auto &e : ctx->ev_free) cudaEventDestroy(e);
    for (auto &e : ctx->ev_ready) cudaEventDestroy(e);
    for (auto &e : ctx->prof_ev) cudaEventDestroy(e);
    if (ctx->ev_done) cudaEventDestroy(ctx->ev_done);
    for (auto p : ctx->ring) cudaFree(p);
    if (ctx->copy_stream) cudaStreamDestroy(ctx->copy_stream);
    cudaFree(ctx->d_tab_img); cudaFree(ctx->d_gen); cudaFree(ctx->d_pos); cudaFree(ctx->d_counts); cudaFree(ctx->d_local); cudaFree(ctx->d_groups);
    cudaFree(ctx->d_scratch); cudaFree(ctx->d_cand); cudaFree(ctx->d_sb); cudaFree(ctx->d_aux);
    cudaFree(ctx->d_carry[0]); cudaFree(ctx->d_carry[1]); cudaFree(ctx->d_queue); cudaFree(ctx->d_hhist); cudaFree(ctx->d_order);
    cudaFree(ctx->index.tag); cudaFree(ctx->index.key); cudaFree(ctx->index.ready); cudaFree(ctx->index.stats);
    if (ctx->h_pinned) cudaFreeHost(ctx->h_pinned);
    if (ctx->h_flag) cudaFreeHost(ctx->h_flag);
    cudaGetLastError();
    delete ctx;
}

// SBArgs of a one-shot bounded call whose ordered candidate list is ctx->d_cand (capacity ccap,
// count in aux->ncand), with the size-rule scratch for it.
int one_shot_sbargs(shred_ctx *ctx, uint64_t ccap, uint64_t len, uint64_t *d_out, uint64_t cap, uint32_t tile,
                    SBArgs &A) {
    Aux *aux = ctx->d_aux + 0;
    const uint64_t nb = (ccap + SB_B - 1) / SB_B;
    int rc = grow(ctx, ctx->d_sb, ctx->sb_cap, 9 * (nb + 2), "size-rule scratch");
    if (rc) return rc;
    A.cand = ctx->d_cand; A.n_dev = &aux->ncand; A.n_host = 0; A.n_cap = ccap;
    A.minsz = ctx->p.min_size; A.maxsz = ctx->p.max_size; A.end = len; A.fin = 1;
    uint64_t *b = ctx->d_sb;
    A.spec_exit = b; A.spec_cnt = b + (nb + 2); A.entry = b + 2 * (nb + 2); A.offs = b + 3 * (nb + 2);
    A.delta = (int64_t *)(b + 4 * (nb + 2)); A.ok = (uint32_t *)(b + 5 * (nb + 2));
    A.cta_sum = b + 6 * (nb + 2); A.cta_ok = b + 7 * (nb + 2); A.cta_off = b + 8 * (nb + 2);
    A.dst = d_out; A.dst_cap = cap; A.aux = aux; A.tile = tile;
    return SHRED_OK;
}

// One-shot bounded call on a small input: k1 -> k_scatter (ordered candidates) -> sb_one (the
// whole size rule, the state set-up and the call end in one CTA).  Three launches instead of
// eight; the multi-CTA sb_* chain is launch-latency bound at these sizes (1 MiB: 27 us per call).
int chunk_bounded_one(shred_ctx *ctx, Plan &pl, uint64_t len, uint64_t *d_out, uint64_t cap,
                      uint64_t *n_out, cudaStream_t st) {
    Aux *aux = ctx->d_aux + 0;
    int rc;
    if ((rc = launch_detect(ctx, pl, st))) return rc;
    const uint64_t ccap = (uint64_t)pl.nslots * pl.J.cap + 1;
    if ((rc = grow(ctx, ctx->d_cand, ctx->cand_cap, ccap, "candidate list"))) return rc;
    if ((rc = launch_scatter(ctx, pl, ctx->d_cand, ccap, aux, 0, nullptr, st))) return rc;
    SBArgs A{};
    if ((rc = one_shot_sbargs(ctx, ccap, len, d_out, cap, SBO_THREADS, A))) return rc;
    size_t smem = 0;
    if (pl.nslots) {
        uint64_t maxseg = pl.J.map.S;
        if (pl.J.map.head_seg > maxseg) maxseg = pl.J.map.head_seg;
        if (pl.J.map.tail_seg > maxseg) maxseg = pl.J.map.tail_seg;
        if (maxseg > SBD_WIN) maxseg = SBD_WIN;
        smem = (size_t)((maxseg + 31) / 32) * 4;
    }
    if (smem < SBO_SMEM) smem = SBO_SMEM;
    PDL(sb_one, 1, SBO_THREADS, smem, st, pl.J, ctx->dp, ctx->d_gen, pl.nslots, A, n_out, cap);
    LAUNCHED("sb_one");
    return SHRED_OK;
}

int shred_chunk(shred_ctx *ctx, const uint8_t *d_in, uint64_t len, uint64_t *d_out, uint64_t cap,
                uint64_t *n_out, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    int rc = check_out(ctx, d_out, cap, n_out);
    if (rc) return rc;
    if (len && !d_in) return fail(ctx, SHRED_EINVAL, "d_in is NULL");
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    Aux *aux = ctx->d_aux + 0;
    Plan pl;
    if ((rc = plan_job(ctx, pl, d_in, 0, nullptr, 0, 0, len, len))) return rc;
    if (!bounded(ctx)) {
        if ((rc = launch_detect(ctx, pl, st))) return rc;
        return launch_scatter(ctx, pl, d_out, cap, aux, 0, n_out, st);
    }
    // few expected candidates (random-like data fits sb_one's shared-memory form): one CTA runs
    // the whole size rule (exact for any count; dense inputs take its global or sb_dense form)
    if (SB_ONE_MAX_LEN && len <= SB_ONE_MAX_LEN &&
        (long double)len * (long double)hits_per_d(ctx->p) / (long double)ctx->p.divisor <= (long double)SB_ONE_EXPECT)
        return chunk_bounded_one(ctx, pl, len, d_out, cap, n_out, st);
    // the multi-CTA chain: k_scatter resets the size-rule state, the rule's last kernel writes
    // the count (no k_stream_reset / k_call_end launches)
    if ((rc = launch_detect(ctx, pl, st))) return rc;
    const uint64_t ccap = (uint64_t)pl.nslots * pl.J.cap + 1;
    if ((rc = grow(ctx, ctx->d_cand, ctx->cand_cap, ccap, "candidate list"))) return rc;
    if ((rc = launch_scatter(ctx, pl, ctx->d_cand, ccap, aux, 0, nullptr, st, 1))) return rc;
    return launch_size_bound(ctx, ctx->d_cand, &aux->ncand, 0, ccap, len, 1, d_out, cap, aux, &pl, st, n_out);
}

int shred_candidates_range(shred_ctx *ctx, const uint8_t *d_in, uint64_t halo, uint64_t start,
                           uint64_t len, uint64_t total_len, uint64_t *d_out, uint64_t cap,
                           uint64_t *n_out, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    int rc = check_out(ctx, d_out, cap, n_out);
    if (rc) return rc;
    const uint64_t want = start < (uint64_t)ctx->p.window - 1u ? start : (uint64_t)ctx->p.window - 1u;
    if (halo != want) return fail(ctx, SHRED_EINVAL, "halo must be min(w-1, start) = %llu", (unsigned long long)want);
    if (start + len > total_len) return fail(ctx, SHRED_EINVAL, "start + len > total_len");
    if ((len || halo) && !d_in) return fail(ctx, SHRED_EINVAL, "d_in is NULL");
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    Aux *aux = ctx->d_aux + 0;
    Plan pl;
    if ((rc = plan_job(ctx, pl, d_in, start - halo, nullptr, 0, start, start + len, total_len))) return rc;
    if ((rc = launch_detect(ctx, pl, st))) return rc;
    return launch_scatter(ctx, pl, d_out, cap, aux, 0, n_out, st);
}

int shred_size_bound(shred_ctx *ctx, const uint64_t *d_cand, uint64_t n_cand, uint64_t total_len,
                     uint64_t *d_out, uint64_t cap, uint64_t *n_out, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    int rc = check_out(ctx, d_out, cap, n_out);
    if (rc) return rc;
    if (n_cand && !d_cand) return fail(ctx, SHRED_EINVAL, "d_cand is NULL");
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    Aux *aux = ctx->d_aux + 0;
    PDL(k_stream_reset, 1, 1, 0, st, aux);
    LAUNCHED("k_stream_reset");
    if ((rc = launch_size_bound(ctx, d_cand, nullptr, n_cand, n_cand, total_len, 1, d_out, cap, aux,
                                nullptr, st))) return rc;
    PDL(k_call_end, 1, 1, 0, st, aux, n_out, cap, nullptr);
    LAUNCHED("k_call_end");
    return SHRED_OK;
}

int shred_size_bound_state(shred_ctx *ctx, const uint64_t *d_cand, uint64_t n_cand, uint64_t end,
                           int fin, const uint64_t state_in[2], uint64_t *d_out, uint64_t cap,
                           uint64_t *n_out, uint64_t *d_state_out, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    int rc = check_out(ctx, d_out, cap, n_out);
    if (rc) return rc;
    if ((n_cand && !d_cand) || !state_in || !d_state_out) return fail(ctx, SHRED_EINVAL, "null pointer");
    if (state_in[0] > end) return fail(ctx, SHRED_EINVAL, "entry state beyond the range end");
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    Aux *aux = ctx->d_aux + 0;
    PDL(k_state_in, 1, 1, 0, st, aux, state_in[0], state_in[1] ? 1ull : 0ull);
    LAUNCHED("k_state_in");
    if ((rc = launch_size_bound(ctx, d_cand, nullptr, n_cand, n_cand, end, fin ? 1 : 0, d_out, cap, aux,
                                nullptr, st))) return rc;
    PDL(k_state_out, 1, 1, 0, st, aux, d_state_out, n_out, cap);
    LAUNCHED("k_state_out");
    return SHRED_OK;
}

int shred_size_bound_state_dev(shred_ctx *ctx, const uint64_t *d_cand, const uint64_t *d_n_cand,
                               uint64_t n_cand_max, uint64_t end, int fin, const uint64_t *d_state_in,
                               uint64_t *d_out, uint64_t cap, uint64_t *n_out, uint64_t *d_state_out,
                               shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    int rc = check_out(ctx, d_out, cap, n_out);
    if (rc) return rc;
    if (!d_n_cand || (n_cand_max && !d_cand) || !d_state_in || !d_state_out)
        return fail(ctx, SHRED_EINVAL, "null pointer");
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    Aux *aux = ctx->d_aux + 0;
    PDL(k_state_in_dev, 1, 1, 0, st, aux, d_state_in);
    LAUNCHED("k_state_in_dev");
    if ((rc = launch_size_bound(ctx, d_cand, d_n_cand, 0, n_cand_max, end, fin ? 1 : 0, d_out, cap, aux,
                                nullptr, st))) return rc;
    PDL(k_state_out, 1, 1, 0, st, aux, d_state_out, n_out, cap);
    LAUNCHED("k_state_out");
    return SHRED_OK;
}

// ---------------------------------------------------------------------------- streaming
int shred_set_ring(shred_ctx *ctx, int slots, uint64_t slot_bytes) {
    if (!ctx) return SHRED_EINVAL;
    if (slots < 1 || slots > 4 || slot_bytes < 4096) return fail(ctx, SHRED_EINVAL, "ring: 1..4 slots of >= 4096 B");
    if (ctx->pos != 0) return fail(ctx, SHRED_ESTATE, "ring can only change between streams");
    DevGuard g(ctx->device);
    if (ctx->copy_stream) cudaStreamSynchronize(ctx->copy_stream);
    cudaDeviceSynchronize();
    for (auto p : ctx->ring) cudaFree(p);
    for (auto &e : ctx->ev_free) cudaEventDestroy(e);
    for (auto &e : ctx->ev_ready) cudaEventDestroy(e);
    ctx->ring.clear(); ctx->ev_free.clear(); ctx->ev_ready.clear();
    ctx->ring_n = slots; ctx->ring_bytes = slot_bytes; ctx->ring_next = 0;
    return SHRED_OK;
}

namespace {
int ensure_ring(shred_ctx *ctx) {
    if (!ctx->ring.empty()) return SHRED_OK;
    for (int i = 0; i < ctx->ring_n; ++i) {
        uint8_t *p = nullptr;
        if (cudaMalloc(&p, ctx->ring_bytes) != cudaSuccess) { cudaGetLastError(); return fail(ctx, SHRED_ENOMEM, "ring slot alloc"); }
        ctx->ring.push_back(p);
        cudaEvent_t a, b;
        cudaEventCreateWithFlags(&a, cudaEventDisableTiming);
        cudaEventCreateWithFlags(&b, cudaEventDisableTiming);
        ctx->ev_free.push_back(a); ctx->ev_ready.push_back(b);
    }
    return SHRED_OK;
}

// Process stream bytes [ctx->pos, ctx->pos + len) that are resident at device pointer `src`.
int feed_device_piece(shred_ctx *ctx, const uint8_t *src, uint64_t len, uint64_t *d_out, uint64_t cap,
                      cudaStream_t st) {
    Aux *aux = ctx->d_aux + 1;
    const uint8_t *prefix = ctx->d_carry[ctx->carry_idx];
    int rc = run_piece(ctx, aux, src, ctx->pos, prefix, ctx->carry_len, ctx->pos, ctx->pos + len,
                       ~0ull, 0, d_out, cap, st);
    if (rc) return rc;
    const uint32_t keep = ctx->p.window - 1u;
    uint8_t *nc = ctx->d_carry[ctx->carry_idx ^ 1];
    PDL(k_carry, 1, 256, 0, st, prefix, ctx->carry_len, src, len, nc, keep);
    LAUNCHED("k_carry");
    ctx->carry_idx ^= 1;
    const uint64_t tot = (uint64_t)ctx->carry_len + len;
    ctx->carry_len = (uint32_t)(tot < keep ? tot : keep);
    ctx->pos += len;
    return SHRED_OK;
}
}  // namespace

int shred_feed(shred_ctx *ctx, const void *in, uint64_t len, uint64_t *d_out, uint64_t cap,
               uint64_t *n_out, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    // an earlier streaming call overflowed its output (observed once that call completed)
    if (*(volatile uint64_t *)ctx->h_flag) ctx->sticky = SHRED_ECAPACITY;
    if (ctx->sticky) return fail(ctx, ctx->sticky, "sticky error from an earlier call; shred_reset first");
    int rc = check_out(ctx, d_out, cap, n_out);
    if (rc) return rc;
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    Aux *aux = ctx->d_aux + 1;
    PDL(k_call_begin, 1, 1, 0, st, aux);
    LAUNCHED("k_call_begin");
    if (len) {
        if (!in) return fail(ctx, SHRED_EINVAL, "in is NULL");
        const int kind = ptr_kind(in);
        if (kind == 0) return fail(ctx, SHRED_EINVAL, "input must be device or page-locked host memory");
        if (kind == 1) {
            if ((rc = feed_device_piece(ctx, (const uint8_t *)in, len, d_out, cap, st))) return rc;
        } else {
            if ((rc = ensure_ring(ctx))) return rc;
            // Pieces of <= one slot.  The H2D copy of piece p+ring-1 is enqueued on the copy
            // stream before piece p is processed, so transfers overlap the chunking (bounded
            // mode too: its size-rule state stays on the device, nothing waits on the host).
            const uint8_t *h = (const uint8_t *)in;
            const uint64_t npieces = (len + ctx->ring_bytes - 1) / ctx->ring_bytes;
            const int R = ctx->ring_n;
            auto slot_of = [&](uint64_t q) { return (int)((ctx->ring_next + q) % (uint64_t)R); };
            auto issue_copy = [&](uint64_t q) -> int {
                const uint64_t off = q * ctx->ring_bytes;
                const uint64_t n = (len - off) < ctx->ring_bytes ? (len - off) : ctx->ring_bytes;
                const int sl = slot_of(q);
                CK(cudaStreamWaitEvent(ctx->copy_stream, ctx->ev_free[sl], 0), "wait slot free");
                CK(cudaMemcpyAsync(ctx->ring[sl], h + off, n, cudaMemcpyHostToDevice, ctx->copy_stream), "H2D");
                CK(cudaEventRecord(ctx->ev_ready[sl], ctx->copy_stream), "record ready");
                return SHRED_OK;
            };
            uint64_t issued = 0;
            for (; issued < npieces && issued < (uint64_t)(R > 1 ? R - 1 : 1); ++issued)
                if ((rc = issue_copy(issued))) return rc;
            for (uint64_t q = 0; q < npieces; ++q) {
                if (R > 1 && issued < npieces && issued <= q + (uint64_t)(R - 1)) {
                    if ((rc = issue_copy(issued))) return rc;
                    ++issued;
                }
                const uint64_t off = q * ctx->ring_bytes;
                const uint64_t n = (len - off) < ctx->ring_bytes ? (len - off) : ctx->ring_bytes;
                const int sl = slot_of(q);
                CK(cudaStreamWaitEvent(st, ctx->ev_ready[sl], 0), "wait ready");
                if ((rc = feed_device_piece(ctx, ctx->ring[sl], n, d_out, cap, st))) return rc;
                CK(cudaEventRecord(ctx->ev_free[sl], st), "record free");
                if (R == 1 && issued < npieces) { if ((rc = issue_copy(issued))) return rc; ++issued; }
            }
            ctx->ring_next = slot_of(npieces);
        }
    }
    PDL(k_call_end, 1, 1, 0, st, aux, n_out, cap, ctx->d_flag);
    LAUNCHED("k_call_end");
    return SHRED_OK;
}

int shred_flush(shred_ctx *ctx, uint64_t *d_out, uint64_t cap, uint64_t *n_out, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    int rc = check_out(ctx, d_out, cap, n_out);
    if (rc) return rc;
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    // Every forced cut strictly inside the stream was emitted by the last feed; a cut held at
    // exactly the stream end is dropped (c = N is never a cut, reading Q11).
    PDL(k_stream_reset, 1, 1, 0, st, ctx->d_aux + 1);
    LAUNCHED("k_stream_reset");
    PDL(k_write_u64, 1, 1, 0, st, n_out, 0);
    LAUNCHED("k_write_u64");
    ctx->pos = 0; ctx->carry_len = 0; ctx->carry_idx = 0;
    return SHRED_OK;
}

int shred_reset(shred_ctx *ctx) {
    if (!ctx) return SHRED_EINVAL;
    DevGuard g(ctx->device);
    if (ctx->copy_stream) cudaStreamSynchronize(ctx->copy_stream);
    cudaDeviceSynchronize();
    cudaMemset(ctx->d_aux + 1, 0, sizeof(Aux));
    cudaDeviceSynchronize();
    ctx->pos = 0; ctx->carry_len = 0; ctx->carry_idx = 0; ctx->sticky = SHRED_OK;
    ctx->h_flag[0] = 0;
    return SHRED_OK;
}

int shred_hash_chunks_batch(shred_ctx *ctx, const shred_hash_job *jobs, int njobs, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    if (njobs < 0 || (njobs && !jobs)) return fail(ctx, SHRED_EINVAL, "jobs is NULL");
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    for (int j0 = 0; j0 < njobs; j0 += HASH_MAX_JOBS) {      // launches of up to HASH_MAX_JOBS buffers
        HashJobs H{};
        uint64_t tot = 0;
        for (int j = j0; j < njobs && H.n < HASH_MAX_JOBS; ++j) {
            const shred_hash_job &q = jobs[j];
            if (!q.d_ncuts || (q.len && !q.d_in) || (q.max_chunks && !q.d_digests))
                return fail(ctx, SHRED_EINVAL, "job %d: null pointer", j);
            if (((uintptr_t)q.d_digests & 15u) != 0) return fail(ctx, SHRED_EINVAL, "job %d: d_digests must be 16-byte aligned", j);
            if (!q.len || !q.max_chunks) continue;
            H.base[H.n] = tot;
            H.job[H.n] = HashJob{q.d_in, q.len, q.d_cuts, q.d_ncuts, q.d_digests, q.max_chunks};
            tot += q.max_chunks;
            ++H.n;
        }
        if (!H.n) continue;
        H.base[H.n] = tot;
        if (tot > 0xFFFFFFFFull) return fail(ctx, SHRED_EINVAL, "more than 2^32 - 1 chunks in one launch");
        int rc = grow(ctx, ctx->d_order, ctx->order_cap, tot, "hash order");
        if (rc) return rc;
        CK(cudaMemsetAsync(ctx->d_hhist, 0, HB * sizeof(uint32_t), st), "hash hist reset");
        const unsigned gs = (unsigned)(ctx->sm_count * 8);
        PDL(k_hash_hist, gs, 256, 0, st, H, ctx->d_hhist);
        LAUNCHED("k_hash_hist");
        PDL(k_hash_scan, 1, HB, 0, st, ctx->d_hhist, ctx->d_queue);
        LAUNCHED("k_hash_scan");
        PDL(k_hash_scatter, gs, 256, 0, st, H, ctx->d_hhist, ctx->d_order);
        LAUNCHED("k_hash_scatter");
        // one warp per SM sub-partition for one buffer (its longest chunk's warp keeps a whole
        // sub-partition); two for a batch, whose work hides the long chains anyway
        // (profiles/r02_hash_ab.txt: 3 x 1 GiB 548 -> 627 GB/s, one buffer 290 -> 242 GB/s)
        const unsigned hctas = (unsigned)(ctx->sm_count * SHRED_HASH_CTAS_PER_SM * (H.n > 1 ? 2 : 1));
        if (SHRED_HASH_WS && (H.n == 1 || SHRED_HASH_WS_BATCH)) {
            // one buffer: the warp-specialised kernel (schedule and rounds on two SM sub-partitions)
            k_hash_chunks_ws<<<(unsigned)ctx->sm_count, HWS_THREADS, HWS_SMEM, st>>>(H, ctx->d_order, ctx->d_queue, 1u);
        } else {
#if SHRED_HASH_NOPDL
            k_hash_chunks<<<hctas, SHRED_HASH_THREADS, 0, st>>>(H, ctx->d_order, ctx->d_queue, 1u);
#else
            PDL(k_hash_chunks, hctas, SHRED_HASH_THREADS, 0, st, H, ctx->d_order, ctx->d_queue, 1u);
#endif
        }
        LAUNCHED("k_hash_chunks");
    }
    return SHRED_OK;
}

int shred_hash_chunks(shred_ctx *ctx, const uint8_t *d_in, uint64_t len, const uint64_t *d_cuts,
                      const uint64_t *d_ncuts, uint8_t *d_digests, uint64_t max_chunks,
                      shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    if (max_chunks > 0xFFFFFFFFull) return fail(ctx, SHRED_EINVAL, "max_chunks must be < 2^32");
    const shred_hash_job j{d_in, len, d_cuts, d_ncuts, d_digests, max_chunks};
    return shred_hash_chunks_batch(ctx, &j, 1, stream);
}

int shred_index_reset(shred_ctx *ctx, uint64_t capacity) {
    if (!ctx || capacity == 0 || capacity > (1ull << 36)) return SHRED_EINVAL;
    DevGuard g(ctx->device);
    uint64_t cap = 1024;
    while (cap < 2 * capacity) cap <<= 1;
    cudaDeviceSynchronize();
    DedupTable &T = ctx->index;
    if (T.cap != cap) {
        cudaFree(T.tag); cudaFree(T.key); cudaFree(T.ready);
        T.tag = nullptr; T.key = nullptr; T.ready = nullptr; T.cap = 0;
        if (cudaMalloc(&T.tag, cap * 8) != cudaSuccess || cudaMalloc(&T.key, cap * 32) != cudaSuccess ||
            cudaMalloc(&T.ready, cap * 4) != cudaSuccess) {
            cudaGetLastError();
            return fail(ctx, SHRED_ENOMEM, "index: cudaMalloc failed for %llu slots", (unsigned long long)cap);
        }
        T.cap = cap;
    }
    if (!T.stats && cudaMalloc(&T.stats, 64) != cudaSuccess) { cudaGetLastError(); return SHRED_ENOMEM; }
    // cudaMemset runs on the legacy default stream and does not block the host; the call has no
    // stream argument, so it completes the clear before returning (a following insert on a
    // non-blocking stream must not see stale slots: ADVICE r01)
    if (cudaMemset(T.tag, 0, cap * 8) != cudaSuccess || cudaMemset(T.ready, 0, cap * 4) != cudaSuccess ||
        cudaMemset(T.stats, 0, 64) != cudaSuccess || cudaDeviceSynchronize() != cudaSuccess)
        return fail(ctx, SHRED_ECUDA, "index reset");
    return SHRED_OK;
}

int shred_index_insert(shred_ctx *ctx, const uint8_t *d_digests, const uint64_t *d_cuts,
                       const uint64_t *d_ncuts, uint64_t len, uint64_t max_chunks,
                       uint8_t *d_new_flags, shred_stream_t stream) {
    if (!ctx) return SHRED_EINVAL;
    if (!ctx->index.cap) return fail(ctx, SHRED_ESTATE, "shred_index_reset first");
    if (!d_ncuts || (max_chunks && !d_digests)) return fail(ctx, SHRED_EINVAL, "null pointer");
    if (((uintptr_t)d_digests & 15u) != 0) return fail(ctx, SHRED_EINVAL, "d_digests must be 16-byte aligned");
    if (!len || !max_chunks) return SHRED_OK;
    DevGuard g(ctx->device);
    cudaStream_t st = (cudaStream_t)stream;
    StreamOrder so(ctx, st);
    PDL(k_dedup_insert, ctx->sm_count * 8, 256, 0, st, ctx->index, d_digests, d_cuts, d_ncuts, len, max_chunks,
                                                      d_new_flags);
    LAUNCHED("k_dedup_insert");
    return SHRED_OK;
}

int shred_index_stats(shred_ctx *ctx, uint64_t stats[4]) {
    if (!ctx || !stats) return SHRED_EINVAL;
    if (!ctx->index.stats) { for (int i = 0; i < 4; ++i) stats[i] = 0; return SHRED_OK; }
    DevGuard g(ctx->device);
    CK(cudaDeviceSynchronize(), "index stats sync");
    CK(cudaMemcpy(stats, ctx->index.stats, 32, cudaMemcpyDeviceToHost), "index stats");
    return SHRED_OK;
}

int shred_check_params(const shred_params *p, int *path_out, int *marker_kind_out) {
    const int rc = validate(p, nullptr);
    if (rc) return rc;
    int mk = -1;
    const int path = select_path(p, &mk);
    if (path_out) *path_out = path;
    if (marker_kind_out) *marker_kind_out = mk;
    return SHRED_OK;
}

int shred_debug_plan(int path, int small_ok, int sm_count, uint64_t src_addr, uint64_t p_begin,
                     uint64_t t_begin, uint64_t t_end, uint64_t divisor, uint32_t window, int zero_lead,
                     uint64_t out[16]) {
    if (!out || t_end < t_begin || t_begin < p_begin || sm_count < 1 || divisor < 2 || window < 1 || window > LW_MAX)
        return SHRED_EINVAL;
    const MapShape sh{path == SHRED_PATH_K63 || path == SHRED_PATH_K32, path == SHRED_PATH_K63, small_ok != 0,
                      sm_count, 16u * ((window + 15u) / 16u), zero_lead != 0};
    SlotMap m;
    bool bulk = false, small = false;
    plan_map(sh, src_addr, p_begin, t_begin, t_end, m, bulk, small);
    const uint64_t v[16] = {bulk, small, m.head_start, m.head_seg, m.n_head, m.b0, m.S, m.nrows,
                            m.tail_start, m.tail_seg, m.n_tail, m.nc, m.ngroups, m.rows_cta,
                            slot_cap(m, bulk, divisor, 1, 0), small ? (uint64_t)CfgSmall::NTC
                                                              : (uint64_t)(path == SHRED_PATH_K63 ? CfgK63::NTC : CfgK32::NTC)};
    for (int i = 0; i < 16; ++i) out[i] = v[i];
    return SHRED_OK;
}

int shred_debug_tprod(uint64_t poly, uint32_t *mult, uint32_t *mult_hi) {
    uint32_t m = 0, mh = 0;
    const int ok = tprod_ok(poly, deg64(poly), &m, &mh) ? 1 : 0;
    if (mult) *mult = m;
    if (mult_hi) *mult_hi = mh;
    return ok;
}

int shred_profile(shred_ctx *ctx, int enable) {
    if (!ctx) return SHRED_EINVAL;
    ctx->prof = enable != 0;
    return SHRED_OK;
}

int shred_profile_read(shred_ctx *ctx, double *ms, uint64_t *launches, uint64_t *bytes) {
    if (!ctx || !ms || !launches || !bytes) return SHRED_EINVAL;
    DevGuard g(ctx->device);
    double tot = 0.0;
    for (size_t i = 0; i + 1 < ctx->prof_used; i += 2) {
        CK(cudaEventSynchronize(ctx->prof_ev[i + 1]), "profile sync");
        float t = 0.f;
        CK(cudaEventElapsedTime(&t, ctx->prof_ev[i], ctx->prof_ev[i + 1]), "profile elapsed");
        tot += t;
    }
    *ms = tot; *launches = ctx->prof_used / 2; *bytes = ctx->prof_bytes;
    ctx->prof_used = 0; ctx->prof_bytes = 0;
    return SHRED_OK;
}

int shred_synth_fill(uint8_t *d_buf, uint64_t len, uint64_t seed, uint64_t offset, shred_stream_t stream) {
    if (!len) return SHRED_OK;
    if (!d_buf) return SHRED_EINVAL;
    uint64_t blocks = (len / 16 + 255) / 256;
    if (blocks > 148 * 16) blocks = 148 * 16;
    if (blocks < 1) blocks = 1;
    k_synth_fill<<<(unsigned)blocks, 256, 0, (cudaStream_t)stream>>>(d_buf, len, seed, offset);
    return cudaGetLastError() == cudaSuccess ? SHRED_OK : SHRED_ECUDA;
}

}  // extern "C"

// sha256.cuh — hashing every chunk (dedup step 2,
// "Hashing: This is the process of computing a collision-resistant hash of the chunk").
//
// The paper names no hash function; SHA-256 (FIPS 180-4) is used (reading H1).
// Chunks are [0, c_0), [c_0, c_1), ..., [c_{n-1}, len): n cuts give n+1 chunks (len > 0).
//
// k_hash_chunks: one lane hashes one chunk (Merkle-Damgard is sequential inside a chunk).
// Chunk sizes are roughly exponential, so chunks are first counting-sorted by length
// (k_hash_hist / k_hash_scan / k_hash_scatter, 128-byte buckets, longest first) and warps take
// 32 consecutive sorted chunks at a time: the lanes of a warp have near-equal lengths and the
// longest chunks start first (LPT).  Full blocks are loaded as 17 aligned words realigned with
// funnel shifts; the last one or two blocks of a chunk (0x80 padding + 64-bit length) take a
// byte-wise path.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>
#include "kernels.cuh"

namespace shred {

// The round constants as instruction immediates: sha_k(t) with t a compile-time index of the
// unrolled round loop folds to a constant (a __constant__ table made ptxas load them into
// registers with LDC inside the round loop of the batched kernel: +20 % time, short-scoreboard
// stalls, profiles/r02_hash_ab.txt).
__device__ __forceinline__ constexpr uint32_t sha_k(int t) {
    constexpr uint32_t k[64] = {
    0x428a2f98u, 0x71374491u, 0xb5c0fbcfu, 0xe9b5dba5u, 0x3956c25bu, 0x59f111f1u, 0x923f82a4u, 0xab1c5ed5u,
    0xd807aa98u, 0x12835b01u, 0x243185beu, 0x550c7dc3u, 0x72be5d74u, 0x80deb1feu, 0x9bdc06a7u, 0xc19bf174u,
    0xe49b69c1u, 0xefbe4786u, 0x0fc19dc6u, 0x240ca1ccu, 0x2de92c6fu, 0x4a7484aau, 0x5cb0a9dcu, 0x76f988dau,
    0x983e5152u, 0xa831c66du, 0xb00327c8u, 0xbf597fc7u, 0xc6e00bf3u, 0xd5a79147u, 0x06ca6351u, 0x14292967u,
    0x27b70a85u, 0x2e1b2138u, 0x4d2c6dfcu, 0x53380d13u, 0x650a7354u, 0x766a0abbu, 0x81c2c92eu, 0x92722c85u,
    0xa2bfe8a1u, 0xa81a664bu, 0xc24b8b70u, 0xc76c51a3u, 0xd192e819u, 0xd6990624u, 0xf40e3585u, 0x106aa070u,
    0x19a4c116u, 0x1e376c08u, 0x2748774cu, 0x34b0bcb5u, 0x391c0cb3u, 0x4ed8aa4au, 0x5b9cca4fu, 0x682e6ff3u,
    0x748f82eeu, 0x78a5636fu, 0x84c87814u, 0x8cc70208u, 0x90befffau, 0xa4506cebu, 0xbef9a3f7u, 0xc67178f2u};
    return k[t];
}

__device__ __forceinline__ uint32_t rotr(uint32_t x, int n) { return __funnelshift_r(x, x, n); }

// One SHA-256 compression of the 16 big-endian words W into H.
// The rounds are bound by the ALU pipe of the warp's SM sub-partition (rotates, LOP3 and IADD3
// all issue there: ~21.5 ALU instructions per round at 2 cycles each), and the warps hashing the
// longest chunks set the launch time.  SHRED_SHA_FMA=2 (default) turns every addition into an
// IMAD (x * one + y with a runtime one) on the otherwise idle FMA pipe, leaving ~16 rotate/logic
// ops per round on the ALU: 1 GiB, bounds off 294 -> 396 GB/s, bounded chunks 400 -> 500 GB/s.
// 1 = only two additions per round moved (292 -> 270); 0 = all on the ALU
// (profiles/r01_hash_ab.txt).
#ifndef SHRED_SHA_FMA
#define SHRED_SHA_FMA 2
#endif
__device__ __forceinline__ uint32_t fma_add(uint32_t x, uint32_t one, uint32_t y) {
    return SHRED_SHA_FMA == 1 ? x * one + y : x + y;
}

template <int SHA_FMA = SHRED_SHA_FMA>
__device__ __forceinline__ void sha256_compress(uint32_t (&H)[8], uint32_t (&W)[16], uint32_t one) {
    uint32_t a = H[0], b = H[1], c = H[2], d = H[3], e = H[4], f = H[5], g = H[6], h = H[7];
#pragma unroll
    for (int t = 0; t < 64; ++t) {
        uint32_t w;
        if (t < 16) {
            w = W[t];
        } else {
            const uint32_t w15 = W[(t - 15) & 15], w2 = W[(t - 2) & 15];
            const uint32_t s0 = rotr(w15, 7) ^ rotr(w15, 18) ^ (w15 >> 3);
            const uint32_t s1 = rotr(w2, 17) ^ rotr(w2, 19) ^ (w2 >> 10);
            if (SHA_FMA == 2)
                w = W[t & 15] = s1 * one + (s0 * one + (W[t & 15] * one + W[(t - 7) & 15]));
            else
                w = W[t & 15] = fma_add(W[t & 15], one, W[(t - 7) & 15]) + s0 + s1;
        }
        const uint32_t S1 = rotr(e, 6) ^ rotr(e, 11) ^ rotr(e, 25);
        const uint32_t S0 = rotr(a, 2) ^ rotr(a, 13) ^ rotr(a, 22);
        const uint32_t ch = (e & f) ^ (~e & g);
        const uint32_t mj = (a & b) ^ (a & c) ^ (b & c);
        if (SHA_FMA == 2) {                // every addition an IMAD (x * one + y): ALU keeps the logic
            const uint32_t t1 = (ch * one + (S1 * one + (w * one + (h * one + sha_k(t)))));
            h = g; g = f; f = e; e = d * one + t1; d = c; c = b; b = a; a = mj * one + (S0 * one + t1);
        } else {
            const uint32_t hkw = fma_add(h, one, fma_add(w, one, sha_k(t)));
            const uint32_t t1 = hkw + S1 + ch;
            h = g; g = f; f = e; e = d + t1; d = c; c = b; b = a; a = t1 + S0 + mj;
        }
    }
    H[0] += a; H[1] += b; H[2] += c; H[3] += d; H[4] += e; H[5] += f; H[6] += g; H[7] += h;
}

__device__ __forceinline__ void sha256_init(uint32_t (&H)[8]) {
    H[0] = 0x6a09e667u; H[1] = 0xbb67ae85u; H[2] = 0x3c6ef372u; H[3] = 0xa54ff53au;
    H[4] = 0x510e527fu; H[5] = 0x9b05688cu; H[6] = 0x1f83d9abu; H[7] = 0x5be0cd19u;
}

// Block `blk` of the padded message of chunk [a, a+L) (L bytes) into big-endian words W.
__device__ __forceinline__ void sha256_block(const uint8_t *__restrict__ in, uint64_t in_len, uint64_t a,
                                             uint64_t L, uint64_t blk, uint32_t (&W)[16]) {
    const uint64_t m0 = blk * 64;                     // message offset of the block
    // word alignment of the ABSOLUTE address (in itself may be unaligned, e.g. a slice x[1:]);
    // an aligned word that holds a byte of [in, in + in_len) lies inside the same allocation
    const uintptr_t pa = reinterpret_cast<uintptr_t>(in) + a + m0;
    const uintptr_t wa = pa & ~(uintptr_t)3;
    const uintptr_t lim = (reinterpret_cast<uintptr_t>(in) + in_len + 3) & ~(uintptr_t)3;
    if (m0 + 64 <= L && wa + 68 <= lim) {             // full block, 17 aligned words in bounds
        const uint32_t *src = reinterpret_cast<const uint32_t *>(wa);
        const uint32_t sh = (uint32_t)(pa & 3) * 8;
        uint32_t prev = __ldg(src);
#pragma unroll
        for (int k = 0; k < 16; ++k) {
            const uint32_t nxt = __ldg(src + k + 1);
            const uint32_t le = __funnelshift_r(prev, nxt, sh);   // 4 stream bytes, little-endian
            W[k] = __byte_perm(le, 0, 0x0123);                    // big-endian word
            prev = nxt;
        }
        return;
    }
    // a padded tail block: the message words by the same aligned loads (only words that start
    // inside the buffer are read), the bytes at or past L replaced by the padding: 0x80 at byte
    // L, zeros, the 64-bit bit length in the last block's words 14-15 (FIPS 180-4 §5.1.1).
    // Round 1 built these blocks a byte at a time with one dependent global load per byte.
    const uint64_t nblk = (L + 9 + 63) / 64;          // blocks of the padded message
    const int64_t valid = (int64_t)L - (int64_t)m0;   // message bytes in this block (may be <= 0)
    const uint32_t sh = (uint32_t)(pa & 3) * 8;
    const uint32_t *src = reinterpret_cast<const uint32_t *>(wa);
    uint32_t prev = (valid > 0 && wa < lim) ? __ldg(src) : 0u;
#pragma unroll
    for (int k = 0; k < 16; ++k) {
        const uintptr_t na = wa + 4u * (uint32_t)(k + 1);
        const uint32_t nxt = (valid > 4 * k && na < lim) ? __ldg(src + k + 1) : 0u;
        uint32_t be = __byte_perm(__funnelshift_r(prev, nxt, sh), 0, 0x0123);   // big-endian word
        prev = nxt;
        const int64_t nv = valid - 4 * k;                                        // message bytes in it
        if (nv < 4) {
            be = nv <= 0 ? 0u : (be & (0xFFFFFFFFu << (32 - 8 * (int)nv)));
            if (nv >= 0) be |= 0x80u << (24 - 8 * (int)nv);                      // the 0x80 byte
        }
        W[k] = be;
    }
    if (blk + 1 == nblk) {
        const uint64_t bits = L * 8;
        W[14] = (uint32_t)(bits >> 32);
        W[15] = (uint32_t)bits;
    }
}

// ---- length-sorted work list (LPT): chunk sizes are ~exponential, so lanes of one warp must
// hash chunks of similar length or the warp idles on its longest lane.  A counting sort by
// length bucket (descending) makes warps take 32 consecutive similar-length chunks, longest
// first.
constexpr int HB = 1024;                 // length buckets of 128 bytes; the last holds >= 128 KiB

__device__ __forceinline__ uint32_t hash_bucket(uint64_t L) {
    const uint64_t k = L >> 7;
    return (uint32_t)(HB - 1 - (k < (uint64_t)(HB - 1) ? k : (uint64_t)(HB - 1)));   // descending
}

// A batch of buffers hashed by one launch sequence (shred_hash_chunks_batch): job b's chunks
// take global indices [base[b], base[b] + max_chunks_b); one length-sorted work list spans all of
// them, so the longest chunks of every buffer start first and the tail of one buffer overlaps
// the bulk of the others (one buffer alone is bound by its longest chunk, DESIGN.md §5b f2).
constexpr int HASH_MAX_JOBS = 16;
struct HashJob {
    const uint8_t *in; uint64_t len;
    const uint64_t *cuts; const uint64_t *n_cuts;   // device count of cuts
    uint8_t *digests; uint64_t max_chunks;
};
struct HashJobs {
    int n;
    uint64_t base[HASH_MAX_JOBS + 1];               // prefix of max_chunks (global index space)
    HashJob job[HASH_MAX_JOBS];
};

__device__ __forceinline__ void chunk_bounds(const uint64_t *cuts, uint64_t ncut, uint64_t len, uint64_t i,
                                             uint64_t &a, uint64_t &b) {
    a = i ? cuts[i - 1] : 0;
    b = i < ncut ? cuts[i] : len;
}
// global index g -> (job, chunk); false if g is beyond the job's true chunk count
__device__ __forceinline__ bool hash_locate(const HashJobs &H, uint64_t g, int &jb, uint64_t &i) {
    jb = 0;
    while (jb + 1 < H.n && g >= H.base[jb + 1]) ++jb;
    i = g - H.base[jb];
    const HashJob &J = H.job[jb];
    const uint64_t nc = J.len ? min(*J.n_cuts + 1, J.max_chunks) : 0;
    return i < nc;
}

__global__ void k_hash_hist(HashJobs H, uint32_t *hist) {
    pdl_entry();
    const uint64_t tot = H.base[H.n];
    for (uint64_t g = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; g < tot; g += (uint64_t)gridDim.x * blockDim.x) {
        int jb; uint64_t i, a, b;
        if (!hash_locate(H, g, jb, i)) continue;
        chunk_bounds(H.job[jb].cuts, *H.job[jb].n_cuts, H.job[jb].len, i, a, b);
        atomicAdd(&hist[hash_bucket(b - a)], 1u);
    }
}

// One CTA: exclusive scan of the HB bucket counts (in place) and reset of the work queue; the
// total number of chunks goes to queue[1] (the workers' bound).
__global__ void __launch_bounds__(HB) k_hash_scan(uint32_t *hist, unsigned long long *queue) {
    pdl_entry();
    __shared__ uint32_t ws[33];
    const uint32_t v = hist[threadIdx.x];
    uint32_t tot;
    const uint32_t off = block_exscan(v, HB, 1, ws, &tot);
    hist[threadIdx.x] = off;
    if (threadIdx.x == 0) { queue[0] = 0; queue[1] = tot; }
}

__global__ void k_hash_scatter(HashJobs H, uint32_t *offs, uint32_t *order) {
    pdl_entry();
    const uint64_t tot = H.base[H.n];
    for (uint64_t g = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; g < tot; g += (uint64_t)gridDim.x * blockDim.x) {
        int jb; uint64_t i, a, b;
        if (!hash_locate(H, g, jb, i)) continue;
        chunk_bounds(H.job[jb].cuts, *H.job[jb].n_cuts, H.job[jb].len, i, a, b);
        order[atomicAdd(&offs[hash_bucket(b - a)], 1u)] = (uint32_t)g;
    }
}

__device__ __forceinline__ void sha256_store(uint8_t *digests, uint64_t chunk, const uint32_t (&H)[8]) {
    uint4 *o = reinterpret_cast<uint4 *>(digests + chunk * 32);
    o[0] = make_uint4(__byte_perm(H[0], 0, 0x0123), __byte_perm(H[1], 0, 0x0123),
                      __byte_perm(H[2], 0, 0x0123), __byte_perm(H[3], 0, 0x0123));
    o[1] = make_uint4(__byte_perm(H[4], 0, 0x0123), __byte_perm(H[5], 0, 0x0123),
                      __byte_perm(H[6], 0, 0x0123), __byte_perm(H[7], 0, 0x0123));
}

// Hash every chunk of every job.  Job b: nchunks = (*n_cuts + 1 if len > 0 else 0), chunk i ends
// at cuts[i] (i < n) or len; digests: 32 bytes per chunk (the SHA-256 digest bytes in order).
// Warps take 32 consecutive entries of the length-sorted `order` at a time from `queue`.
// Launched with one warp per SM sub-partition: the sequential SHA chain of the longest chunks
// bounds the run, so few warps (each issuing at full rate) beat many (profiles/r01_hash_ab.txt).
__global__ void __launch_bounds__(256)
k_hash_chunks(HashJobs Hj, const uint32_t *__restrict__ order, unsigned long long *queue, uint32_t one) {
    pdl_entry();
    const uint64_t nc = queue[1];
    const int lane = threadIdx.x & 31;
    uint32_t H[8], W[16];
    while (true) {
        unsigned long long base = 0;
        if (lane == 0) base = atomicAdd(queue, 32ull);
        base = __shfl_sync(0xffffffffu, base, 0);
        if (base >= nc) break;
        const uint64_t j = base + (uint64_t)lane;
        if (j < nc) {
            int jb; uint64_t chunk;
            hash_locate(Hj, order[j], jb, chunk);
            const HashJob &J = Hj.job[jb];
            const uint8_t *in = J.in;
            const uint64_t len = J.len;
            uint64_t a, b;
            chunk_bounds(J.cuts, *J.n_cuts, len, chunk, a, b);
            const uint64_t L = b - a, nblk = (L + 9 + 63) / 64;
            sha256_init(H);
            // full blocks: the 17 aligned words of block blk+1 are loaded before block blk is
            // compressed (software pipelining: the load latency hides behind ~1.5K cycles of
            // rounds); the padded tail blocks take the byte path of sha256_block
            // word loads aligned on the ABSOLUTE address (in may be unaligned: ADVICE r01)
            const uintptr_t pa = reinterpret_cast<uintptr_t>(in) + a;
            const uintptr_t lim = (reinterpret_cast<uintptr_t>(in) + len + 3) & ~(uintptr_t)3;
            const uint32_t sh = (uint32_t)(pa & 3) * 8;
            const uint32_t *src0 = reinterpret_cast<const uint32_t *>(pa & ~(uintptr_t)3);
            uint64_t nfull = L / 64;                               // complete message blocks
            if (nfull && (pa & ~(uintptr_t)3) + 64 * nfull + 4 > lim) --nfull;   // 17th word in bounds
            uint32_t Rw[17];
            if (nfull) {
#pragma unroll
                for (int k = 0; k < 17; ++k) Rw[k] = __ldg(src0 + k);
            }
            for (uint64_t blk = 0; blk < nfull; ++blk) {
#pragma unroll
                for (int k = 0; k < 16; ++k) W[k] = __byte_perm(__funnelshift_r(Rw[k], Rw[k + 1], sh), 0, 0x0123);
                if (blk + 1 < nfull) {
                    const uint32_t *nx = src0 + 16 * (blk + 1);
#pragma unroll
                    for (int k = 0; k < 17; ++k) Rw[k] = __ldg(nx + k);
                }
                sha256_compress(H, W, one);
            }
            for (uint64_t blk = nfull; blk < nblk; ++blk) {
                sha256_block(in, len, a, L, blk, W);
                sha256_compress(H, W, one);
            }
            sha256_store(J.digests, chunk, H);
        }
        __syncwarp();
    }
}

// ---- warp-specialised hashing (one buffer: the longest chunks' chains set the time).  A CTA
// holds HWS_PAIRS pairs of warps.  The schedule warp of a pair takes 32 length-sorted chunks from
// the queue, loads each lane's message blocks and expands them to the 64-word schedule W[0..63]
// (sigma0/sigma1: ~8 ALU ops per round for 48 of the 64 rounds) into a shared ring; the
// compress warp runs only the 64 rounds (S0, S1, Ch, Maj: ~10 ALU ops per round, W read by one
// LDS).  The two warps of a pair sit on different SM sub-partitions (compress warp p on SMSP p,
// its schedule warp on SMSP p+1 mod 4), so once only the longest chunks are left their chain
// runs on one sub-partition's ALU with the schedule work on another's.  mbarriers per pair:
// full/free per W slot, info_full/info_free for the batch description.
#ifndef SHRED_HWS_PAIRS
#define SHRED_HWS_PAIRS 4
#endif
constexpr int HWS_PAIRS = SHRED_HWS_PAIRS;
constexpr int HWS_THREADS = 64 * HWS_PAIRS;
#ifndef SHRED_HWS_SLOTS
#define SHRED_HWS_SLOTS 4
#endif
constexpr int HWS_SLOTS = SHRED_HWS_SLOTS;   // W ring depth (blocks the schedule warp may run ahead)
struct HwsPair {
    unsigned long long bar[2 * HWS_SLOTS + 2];   // full[slots], free[slots], info_full, info_free
    uint64_t dig[32];                       // per lane: digest destination (0 = no chunk)
    uint32_t nblk[32];                      // per lane: blocks of the padded message
    uint32_t nmax;                          // the batch's longest; 0xFFFFFFFF = no more work
};
// Every lane arrives on the pair's mbarriers (count 32), so each lane's own shared-memory writes
// (W words, batch fields) are released by its own arrive and acquired by the waiting warp: the
// ordering needs no argument about __syncwarp cumulativity, and compute-sanitizer racecheck
// models it (a __syncwarp + one elected arrive reported 200 false hazards).
#ifndef SHRED_HWS_ALL_ARRIVE
#define SHRED_HWS_ALL_ARRIVE 1
#endif
#if SHRED_HWS_ALL_ARRIVE
constexpr uint32_t HWS_ARRIVALS = 32;
#define HWS_ARRIVE(bar) mbar_arrive(bar)
#else
constexpr uint32_t HWS_ARRIVALS = 1;
#define HWS_ARRIVE(bar) do { __syncwarp(); if (lane == 0) mbar_arrive(bar); } while (0)
#endif
#ifndef SHRED_HWS_ADD
#define SHRED_HWS_ADD 0   // compress-round additions on the FMA pipe: 0 none, 1 a's, 2 a's and t1's (A/B)
#endif
constexpr size_t HWS_RING = (size_t)HWS_SLOTS * 64 * 32 * 4;   // bytes of W ring per pair (slots x 64 words x 32 lanes)
constexpr size_t HWS_SMEM = HWS_PAIRS * (HWS_RING + sizeof(HwsPair)) + 128;

__global__ void __launch_bounds__(HWS_THREADS, 1)
k_hash_chunks_ws(HashJobs Hj, const uint32_t *__restrict__ order, unsigned long long *queue, uint32_t one) {
    pdl_entry();
    extern __shared__ __align__(128) uint8_t hws_smem[];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const bool comp = warp < HWS_PAIRS;
    const int pair = comp ? warp : (warp - HWS_PAIRS + HWS_PAIRS - 1) % HWS_PAIRS;
    uint32_t *ring = reinterpret_cast<uint32_t *>(hws_smem + pair * HWS_RING);
    HwsPair &P = reinterpret_cast<HwsPair *>(hws_smem + HWS_PAIRS * HWS_RING)[pair];
    const uint32_t bfull = smem_u32(&P.bar[0]), bfree = smem_u32(&P.bar[HWS_SLOTS]);
    const uint32_t binfo_full = smem_u32(&P.bar[2 * HWS_SLOTS]), binfo_free = smem_u32(&P.bar[2 * HWS_SLOTS + 1]);
    if (comp && lane == 0) {
        for (int k = 0; k < 2 * HWS_SLOTS + 2; ++k) mbar_init(smem_u32(&P.bar[k]), HWS_ARRIVALS);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();
    const uint64_t nc = queue[1];
    uint32_t gb = 0;                         // blocks passed through the ring (phase counter)
    if (!comp) {                             // ---- schedule warp
        uint32_t W[16];
        for (uint32_t it = 0;; ++it) {
            if (it > 0) mbar_wait(binfo_free, (it - 1) & 1u);
            unsigned long long base = 0;
            if (lane == 0) base = atomicAdd(queue, 32ull);
            base = __shfl_sync(0xffffffffu, base, 0);
            const uint64_t j = base + (uint64_t)lane;
            // job fields copied to registers (a pointer into the kernel parameters would force a
            // stack copy of them)
            const uint8_t *jin = nullptr;
            uint64_t jlen = 0, a = 0, L = 0, chunk = 0, dig = 0;
            uint32_t nb = 0;
            if (base < nc && j < nc) {
                int jb;
                hash_locate(Hj, order[j], jb, chunk);
                const HashJob &J = Hj.job[jb];
                jin = J.in; jlen = J.len;
                uint64_t b;
                chunk_bounds(J.cuts, *J.n_cuts, J.len, chunk, a, b);
                L = b - a;
                nb = (uint32_t)((L + 9 + 63) / 64);
                dig = reinterpret_cast<uint64_t>(J.digests + chunk * 32);
            }
            uint32_t mx = nb;
#pragma unroll
            for (int d = 16; d; d >>= 1) mx = max(mx, __shfl_xor_sync(0xffffffffu, mx, d));
            P.nblk[lane] = nb;
            P.dig[lane] = dig;
            if (lane == 0) P.nmax = base < nc ? mx : 0xFFFFFFFFu;
            HWS_ARRIVE(binfo_full);
            if (base >= nc) break;
            // full blocks by 17 aligned word loads issued one block ahead (their latency hides
            // behind the previous block's expansion); the padded tail blocks by sha256_block
            const uintptr_t pa = reinterpret_cast<uintptr_t>(jin) + a;
            const uintptr_t lim = (reinterpret_cast<uintptr_t>(jin) + jlen + 3) & ~(uintptr_t)3;
            const uint32_t sh = (uint32_t)(pa & 3) * 8;
            const uint32_t *src0 = reinterpret_cast<const uint32_t *>(pa & ~(uintptr_t)3);
            uint32_t nfull = (uint32_t)(L / 64);
            if (nfull && (pa & ~(uintptr_t)3) + 64ull * nfull + 4 > lim) --nfull;
            uint32_t Rw[17];
            if (nfull) {
#pragma unroll
                for (int k = 0; k < 17; ++k) Rw[k] = __ldg(src0 + k);
            }
            for (uint32_t blk = 0; blk < mx; ++blk, ++gb) {
                const uint32_t slot = gb % HWS_SLOTS;
                if (gb >= HWS_SLOTS) mbar_wait(bfree + 8 * slot, ((gb / HWS_SLOTS) - 1) & 1u);
                if (blk < nb) {
                    if (blk < nfull) {
#pragma unroll
                        for (int k = 0; k < 16; ++k) W[k] = __byte_perm(__funnelshift_r(Rw[k], Rw[k + 1], sh), 0, 0x0123);
                        if (blk + 1 < nfull) {
                            const uint32_t *nx = src0 + 16 * (blk + 1);
#pragma unroll
                            for (int k = 0; k < 17; ++k) Rw[k] = __ldg(nx + k);
                        }
                    } else {
                        sha256_block(jin, jlen, a, L, blk, W);
                    }
                    uint32_t *dst = ring + slot * (64 * 32) + lane;
#pragma unroll
                    for (int t = 0; t < 64; ++t) {
                        uint32_t w;
                        if (t < 16) {
                            w = W[t];
                        } else {
                            const uint32_t w15 = W[(t - 15) & 15], w2 = W[(t - 2) & 15];
                            const uint32_t s0 = rotr(w15, 7) ^ rotr(w15, 18) ^ (w15 >> 3);
                            const uint32_t s1 = rotr(w2, 17) ^ rotr(w2, 19) ^ (w2 >> 10);
                            w = W[t & 15] = s1 + s0 + W[t & 15] + W[(t - 7) & 15];
                        }
                        dst[t * 32] = w;
                    }
                }
                HWS_ARRIVE(bfull + 8 * slot);
            }
        }
        return;
    }
    // ---- compress warp
    for (uint32_t it = 0;; ++it) {
        mbar_wait(binfo_full, it & 1u);
        const uint32_t mx = P.nmax, nb = P.nblk[lane];
        uint8_t *dg = reinterpret_cast<uint8_t *>(P.dig[lane]);
        __syncwarp();
        if (mx == 0xFFFFFFFFu) break;
        uint32_t H[8];
        sha256_init(H);
        for (uint32_t blk = 0; blk < mx; ++blk, ++gb) {
            const uint32_t slot = gb % HWS_SLOTS;
            mbar_wait(bfull + 8 * slot, (gb / HWS_SLOTS) & 1u);
            if (blk < nb) {
                const uint32_t *src = ring + slot * (64 * 32) + lane;
                uint32_t a = H[0], b = H[1], c = H[2], d = H[3], e = H[4], f = H[5], g = H[6], h = H[7];
#pragma unroll
                for (int t = 0; t < 64; ++t) {
                    // The chain e -> e' is S1 (3 rotates + LOP3) then one IADD3: the terms that do
                    // not depend on this round's e or a (h + K + w, and d + h + K + w) are
                    // IMADs off the chain.  This warp runs alone on its sub-partition once only
                    // the longest chunks remain, so latency, not ALU throughput, sets its speed
                    // (the all-IMAD additions of k_hash_chunks: ~2.3 K cycles per block here).
                    const uint32_t w = src[t * 32];
                    const uint32_t hkw = w * one + (h * one + sha_k(t));
                    const uint32_t dhkw = d * one + hkw;
                    const uint32_t S1 = rotr(e, 6) ^ rotr(e, 11) ^ rotr(e, 25);
                    const uint32_t S0 = rotr(a, 2) ^ rotr(a, 13) ^ rotr(a, 22);
                    const uint32_t ch = (e & f) ^ (~e & g);
                    const uint32_t mj = (a & b) ^ (a & c) ^ (b & c);
#if SHRED_HWS_ADD == 0
                    const uint32_t t1 = hkw + S1 + ch;
                    h = g; g = f; f = e; e = dhkw + S1 + ch; d = c; c = b; b = a; a = t1 + S0 + mj;
#elif SHRED_HWS_ADD == 1
                    const uint32_t t1 = hkw + S1 + ch;
                    h = g; g = f; f = e; e = dhkw + S1 + ch; d = c; c = b; b = a;
                    a = mj * one + (S0 * one + t1);
#else
                    const uint32_t t1 = S1 * one + (ch * one + hkw);
                    h = g; g = f; f = e; e = dhkw + S1 + ch; d = c; c = b; b = a;
                    a = mj * one + (S0 * one + t1);
#endif
                }
                H[0] += a; H[1] += b; H[2] += c; H[3] += d; H[4] += e; H[5] += f; H[6] += g; H[7] += h;
            }
            HWS_ARRIVE(bfree + 8 * slot);
        }
        if (dg) sha256_store(dg, 0, H);
        HWS_ARRIVE(binfo_free);
    }
}

}  // namespace shred

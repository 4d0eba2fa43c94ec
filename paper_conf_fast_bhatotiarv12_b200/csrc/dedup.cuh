// dedup.cuh — dedup step 3 "Matching" on the GPU (PAPER.md L235-L238:
// "checking if the hash for a chunk already exists in the index.  If it exists then there is a
// duplicate chunk, else the chunk is new and its hash is added to the index").
//
// The index is an open-addressing hash set of 32-byte SHA-256 digests in device memory
// (linear probing, capacity a power of two).  A slot is claimed by a 64-bit CAS of its tag
// (the digest's first 8 bytes | 1; 0 = empty); the claimer writes the full key and then
// publishes the slot (release).  An inserter that meets the same tag waits for the publication
// and compares all 32 bytes.  Exactly one inserter of a given digest sees "new", so the counts
// (new chunks, new bytes) are deterministic; which of two identical chunks of one batch is the
// new one is not.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace shred {

struct DedupTable {
    unsigned long long *tag;    // [cap] 0 = empty, else (first 8 digest bytes) | 1
    uint4 *key;                 // [cap * 2] the 32-byte digests
    uint32_t *ready;            // [cap] 1 once key is written
    uint64_t cap;               // power of two
    unsigned long long *stats;  // [0] chunks inserted, [1] new chunks, [2] new bytes, [3] table full
};

__global__ void k_dedup_insert(DedupTable T, const uint8_t *__restrict__ digests, const uint64_t *cuts,
                               const uint64_t *n_cuts, uint64_t len, uint64_t max_chunks,
                               uint8_t *new_flags) {
    pdl_entry();
    const uint64_t ncut = *n_cuts;
    const uint64_t nc = len ? min(ncut + 1, max_chunks) : 0;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < nc; i += (uint64_t)gridDim.x * blockDim.x) {
        const uint4 *d = reinterpret_cast<const uint4 *>(digests + i * 32);
        const uint4 k0 = d[0], k1 = d[1];
        const unsigned long long tg = (((unsigned long long)k0.y << 32) | k0.x) | 1ull;
        uint64_t slot = (tg >> 1) & (T.cap - 1);
        bool fresh = false, done = false;
        for (uint64_t probe = 0; probe < T.cap && !done; ++probe) {
            const unsigned long long old = atomicCAS(&T.tag[slot], 0ull, tg);
            if (old == 0ull) {                                   // claimed: publish the key
                T.key[2 * slot] = k0;
                T.key[2 * slot + 1] = k1;
                __threadfence();
                atomicExch(&T.ready[slot], 1u);
                fresh = true; done = true;
            } else if (old == tg) {                              // same tag: compare the key
                while (atomicAdd(&T.ready[slot], 0u) == 0u) __nanosleep(32);
                __threadfence();
                const uint4 a0 = T.key[2 * slot], a1 = T.key[2 * slot + 1];
                if (a0.x == k0.x && a0.y == k0.y && a0.z == k0.z && a0.w == k0.w &&
                    a1.x == k1.x && a1.y == k1.y && a1.z == k1.z && a1.w == k1.w) done = true;
            }
            if (!done) slot = (slot + 1) & (T.cap - 1);
        }
        if (!done) atomicAdd(&T.stats[3], 1ull);                 // table full: reported, not inserted
        const uint64_t a = i ? cuts[i - 1] : 0, b = i < ncut ? cuts[i] : len;
        atomicAdd(&T.stats[0], 1ull);
        if (fresh) { atomicAdd(&T.stats[1], 1ull); atomicAdd(&T.stats[2], (unsigned long long)(b - a)); }
        if (new_flags) new_flags[i] = fresh ? 1 : 0;
    }
}

}  // namespace shred

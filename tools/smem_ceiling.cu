// smem_ceiling.cu — measures the B200 shared-memory datapath ceiling that bounds k1_bulk.
//
// The hot loop's per-byte shared-memory work is two data-dependent table lookups (LDS.64 for
// the u64 state, LDS.32 for the u32 state) into a per-lane replicated 64 KiB T|U image, plus
// one LDS.128 of staged input per 16 bytes.  This kernel issues exactly that access mix with
// the same addressing (row t * 256 + lane replica), but without the fingerprint arithmetic and
// with independent (not chained) indices, so it measures what the SMEM datapath alone can
// deliver.  Output: achieved "input bytes per second" if every byte cost exactly that mix, per
// mode, next to wavefront-rate arithmetic (128 B/clk/SM).
//
// Build/run (GPU box): nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o smem_ceiling
//                      tools/smem_ceiling.cu && ./smem_ceiling
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

template <int W>   // W = 8 (u64 lookups, K63) or 4 (u32 lookups, K32)
__global__ void __launch_bounds__(512, 1) lookups(uint32_t *out, int iters) {
    extern __shared__ __align__(16) uint8_t sm[];
    const int tid = threadIdx.x, lane = tid & 31;
    for (int i = tid; i < 65536 / 4 + 512 * 16 / 4; i += blockDim.x)
        reinterpret_cast<uint32_t *>(sm)[i] = i * 2654435761u;
    __syncthreads();
    const uint32_t base = (uint32_t)__cvta_generic_to_shared(sm);
    const uint32_t laneT = base + (W == 8 ? (lane & 15) * 8 : lane * 4);
    const uint32_t laneU = laneT + 128;
    const uint32_t stage = base + 65536 + tid * 16;
    uint32_t x = tid * 747796405u + 1u, acc0 = 0, acc1 = 0;
    for (int it = 0; it < iters; ++it) {
        uint4 d;
        asm volatile("ld.shared.v4.u32 {%0,%1,%2,%3}, [%4];" : "=r"(d.x), "=r"(d.y), "=r"(d.z), "=r"(d.w) : "r"(stage));
        acc0 ^= d.x ^ d.w;
#pragma unroll
        for (int j = 0; j < 16; ++j) {          // 16 "bytes": 2 lookups each, random rows
            x = x * 1664525u + 1013904223u;     // LCG: independent row indices (no chain)
            const uint32_t t = x >> 24, o = (x >> 16) & 255u;
            if (W == 8) {
                uint32_t a, b, c, e;
                asm volatile("ld.shared.v2.u32 {%0,%1}, [%2];" : "=r"(a), "=r"(b) : "r"(laneT + t * 256));
                asm volatile("ld.shared.v2.u32 {%0,%1}, [%2];" : "=r"(c), "=r"(e) : "r"(laneU + o * 256));
                acc0 ^= a ^ c; acc1 ^= b ^ e;
            } else {
                uint32_t a, c;
                asm volatile("ld.shared.u32 %0, [%1];" : "=r"(a) : "r"(laneT + t * 256));
                asm volatile("ld.shared.u32 %0, [%1];" : "=r"(c) : "r"(laneU + o * 256));
                acc0 ^= a ^ c;
            }
        }
    }
    if ((acc0 ^ acc1) == 0x12345678u) out[blockIdx.x * blockDim.x + tid] = acc0;
}

template <int W>
void run(int sms, int clk_khz) {
    const int threads = 512, iters = 4096;
    const size_t smem = 65536 + threads * 16;
    cudaFuncSetAttribute(lookups<W>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    uint32_t *out;
    cudaMalloc(&out, sizeof(uint32_t) * sms * threads);
    lookups<W><<<sms, threads, smem>>>(out, 16);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0); cudaEventCreate(&e1);
    cudaEventRecord(e0);
    lookups<W><<<sms, threads, smem>>>(out, iters);
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms = 0;
    cudaEventElapsedTime(&ms, e0, e1);
    const double bytes = (double)sms * threads * iters * 16;          // "input bytes" processed
    const double wf = (W == 8 ? 4.0 : 2.0) + 4.0 / 16.0;              // wavefronts per 32 lane-bytes
    const double ceil_gbs = 128.0 / (wf * 128.0 / 32.0) * sms * clk_khz * 1e3 / 1e9;
    printf("{\"lookup_bytes\": %d, \"input_GBps_equiv\": %.1f, \"wavefront_ceiling_GBps\": %.1f, "
           "\"ms\": %.3f, \"sms\": %d, \"max_sm_mhz\": %.0f}\n",
           W, bytes / (ms * 1e-3) / 1e9, ceil_gbs, ms, sms, clk_khz / 1e3);
    cudaFree(out);
}

int main() {
    cudaDeviceProp p;
    cudaGetDeviceProperties(&p, 0);
    int clk = 0;
    cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    run<8>(p.multiProcessorCount, clk);
    run<4>(p.multiProcessorCount, clk);
    return 0;
}

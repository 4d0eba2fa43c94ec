// tex_pipe.cu — can a second on-chip data path serve half of k1_bulk<K63>'s table lookups?
//
// k1_bulk<K63> is bound by the L1TEX LSU data pipe: per input byte two 8-byte lookups into a
// replicated shared-memory image (T by the state's top byte, U by the byte leaving the window),
// 4 wavefronts per warp-byte (tools/smem_ceiling.cu: 2,021 GB/s-equivalent at 99.4 % of the
// pipe).  The U lookup does not depend on the state.  This microbenchmark issues the same mix
// with the U lookups moved to other paths, to measure whether they run beside the LDS traffic:
//   mode 0: T LDS.64 + U LDS.64 (the kernel's mix; reference)
//   mode 1: T LDS.64 + U tex1Dfetch<uint2> from a 2 KiB texture (TEX pipe)
//   mode 2: U tex1Dfetch only (the TEX path's own rate)
//   mode 3: T LDS.64 + U ld.global.nc.v2 from a 2 KiB table (L1-resident, LSU global path)
//   mode 4: T LDS.64 + U as two 16-entry halves (U = Ulo[o & 15] ^ Uhi[o >> 4], one 128-B line
//           each) by tex1Dfetch
//   mode 5: T LDS.64 only (half the lookups: the ceiling if U were free)
//   mode 6/7/8: T LDS.64; U by tex1Dfetch for 3/4/6 of every 16 bytes, by LDS.64 for the rest
//           (the two data pipes in parallel)
// Output: one JSON line per mode with the input-byte rate each mix would allow.
//
// Build/run (GPU box): nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o /tmp/tex_pipe
//                      tools/tex_pipe.cu && /tmp/tex_pipe
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

template <int MODE>
__global__ void __launch_bounds__(512, 1) mix(uint32_t *out, int iters, cudaTextureObject_t tex,
                                              cudaTextureObject_t texh, const uint2 *__restrict__ gU) {
    extern __shared__ __align__(16) uint8_t sm[];
    const int tid = threadIdx.x, lane = tid & 31;
    for (int i = tid; i < 65536 / 4 + 512 * 16 / 4; i += blockDim.x)
        reinterpret_cast<uint32_t *>(sm)[i] = i * 2654435761u;
    __syncthreads();
    const uint32_t base = (uint32_t)__cvta_generic_to_shared(sm);
    const uint32_t laneT = base + (lane & 15) * 8;
    const uint32_t laneU = laneT + 128;
    const uint32_t stage = base + 65536 + tid * 16;
    uint32_t x = tid * 747796405u + blockIdx.x, acc0 = 0, acc1 = 0;
    for (int it = 0; it < iters; ++it) {
        uint4 d;
        asm volatile("ld.shared.v4.u32 {%0,%1,%2,%3}, [%4];" : "=r"(d.x), "=r"(d.y), "=r"(d.z), "=r"(d.w) : "r"(stage));
        acc0 ^= d.x ^ d.w;
#pragma unroll
        for (int j = 0; j < 16; ++j) {
            x = x * 1664525u + 1013904223u;
            const uint32_t t = x >> 24, o = (x >> 16) & 255u;
            uint32_t a = 0, b = 0, c = 0, e = 0;
            if (MODE != 2)
                asm volatile("ld.shared.v2.u32 {%0,%1}, [%2];" : "=r"(a), "=r"(b) : "r"(laneT + t * 256));
            if (MODE == 0) {
                asm volatile("ld.shared.v2.u32 {%0,%1}, [%2];" : "=r"(c), "=r"(e) : "r"(laneU + o * 256));
            } else if (MODE == 1 || MODE == 2) {
                const uint2 u = tex1Dfetch<uint2>(tex, (int)o);
                c = u.x; e = u.y;
            } else if (MODE == 3) {
                const uint2 u = __ldg(gU + o);
                c = u.x; e = u.y;
            } else if (MODE >= 6) {
                constexpr int NT = MODE == 6 ? 3 : MODE == 7 ? 4 : 6;
                if (j % 16 < NT) {
                    const uint2 u = tex1Dfetch<uint2>(tex, (int)o);
                    c = u.x; e = u.y;
                } else {
                    asm volatile("ld.shared.v2.u32 {%0,%1}, [%2];" : "=r"(c), "=r"(e) : "r"(laneU + o * 256));
                }
            } else if (MODE == 4) {
                const uint2 u0 = tex1Dfetch<uint2>(texh, (int)(o & 15u));
                const uint2 u1 = tex1Dfetch<uint2>(texh, (int)(16u + (o >> 4)));
                c = u0.x ^ u1.x; e = u0.y ^ u1.y;
            }
            acc0 ^= a ^ c; acc1 ^= b ^ e;
        }
    }
    if ((acc0 ^ acc1) == 0x12345678u) out[blockIdx.x * blockDim.x + tid] = acc0;
}

template <int MODE>
void run(int sms, int clk_khz, cudaTextureObject_t tex, cudaTextureObject_t texh, const uint2 *gU) {
    const int threads = 512, iters = 4096;
    const size_t smem = 65536 + threads * 16;
    cudaFuncSetAttribute(mix<MODE>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    uint32_t *out;
    cudaMalloc(&out, sizeof(uint32_t) * sms * threads);
    mix<MODE><<<sms, threads, smem>>>(out, 16, tex, texh, gU);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0); cudaEventCreate(&e1);
    float best = 1e30f;
    for (int rep = 0; rep < 3; ++rep) {
        cudaEventRecord(e0);
        mix<MODE><<<sms, threads, smem>>>(out, iters, tex, texh, gU);
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
        float ms = 0;
        cudaEventElapsedTime(&ms, e0, e1);
        if (ms < best) best = ms;
    }
    const double bytes = (double)sms * threads * iters * 16;
    printf("{\"mode\": %d, \"input_GBps_equiv\": %.1f, \"ms\": %.3f, \"sms\": %d, \"max_sm_mhz\": %.0f, \"err\": \"%s\"}\n",
           MODE, bytes / (best * 1e-3) / 1e9, best, sms, clk_khz / 1e3, cudaGetErrorString(cudaGetLastError()));
    cudaFree(out);
}

static cudaTextureObject_t make_tex(const uint2 *d, int n) {
    cudaResourceDesc rd = {};
    rd.resType = cudaResourceTypeLinear;
    rd.res.linear.devPtr = const_cast<uint2 *>(d);
    rd.res.linear.desc = cudaCreateChannelDesc<uint2>();
    rd.res.linear.sizeInBytes = sizeof(uint2) * n;
    cudaTextureDesc td = {};
    td.readMode = cudaReadModeElementType;
    cudaTextureObject_t t = 0;
    cudaCreateTextureObject(&t, &rd, &td, nullptr);
    return t;
}

int main() {
    cudaDeviceProp p;
    cudaGetDeviceProperties(&p, 0);
    int clk = 0;
    cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    uint2 h[256];
    for (int i = 0; i < 256; ++i) h[i] = make_uint2(i * 2654435761u, i * 40503u + 7u);
    uint2 *dU, *dH;
    cudaMalloc(&dU, sizeof(h));
    cudaMalloc(&dH, 32 * sizeof(uint2));
    cudaMemcpy(dU, h, sizeof(h), cudaMemcpyHostToDevice);
    cudaMemcpy(dH, h, 32 * sizeof(uint2), cudaMemcpyHostToDevice);
    cudaTextureObject_t tex = make_tex(dU, 256), texh = make_tex(dH, 32);
    run<0>(p.multiProcessorCount, clk, tex, texh, dU);
    run<1>(p.multiProcessorCount, clk, tex, texh, dU);
    run<2>(p.multiProcessorCount, clk, tex, texh, dU);
    run<3>(p.multiProcessorCount, clk, tex, texh, dU);
    run<4>(p.multiProcessorCount, clk, tex, texh, dU);
    run<5>(p.multiProcessorCount, clk, tex, texh, dU);
    run<6>(p.multiProcessorCount, clk, tex, texh, dU);
    run<7>(p.multiProcessorCount, clk, tex, texh, dU);
    run<8>(p.multiProcessorCount, clk, tex, texh, dU);
    return 0;
}

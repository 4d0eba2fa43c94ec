// Pipe assignment and issue rate of the single instructions the k <= 32 hot loop is built from
// (round 2).  Each kernel runs 8 independent dependency chains of one instruction
// form per thread; ncu's sm__inst_executed_pipe_* counters name the pipe, the kernel time the rate.
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o pipe_probe tools/pipe_probe.cu
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

#define CH 8
#define IT 4096

#define KERNEL(NAME, BODY)                                                                   \
    __global__ void NAME(uint32_t *out, uint32_t a, uint32_t b, uint32_t c) {                \
        uint32_t x[CH];                                                                      \
        _Pragma("unroll") for (int j = 0; j < CH; ++j) x[j] = threadIdx.x * (j + 1) + a;     \
        _Pragma("unroll 1") for (int i = 0; i < IT; ++i) {                                   \
            _Pragma("unroll") for (int j = 0; j < CH; ++j) { BODY }                          \
        }                                                                                    \
        uint32_t s = 0;                                                                      \
        _Pragma("unroll") for (int j = 0; j < CH; ++j) s ^= x[j];                             \
        if (s == 0x12345678u) out[threadIdx.x] = s;                                          \
    }

// predicated add of an immediate after a fused LOP3 predicate (the marker test + hit accumulate)
KERNEL(k_lop3p_viadd, asm volatile("{\n .reg .pred p;\n lop3.b32 %0, %0, %1, %2, 0x96;\n"
                                   " setp.ne.u32 p, %0, 0;\n @p add.u32 %0, %0, 3;\n}" : "+r"(x[j]) : "r"(b), "r"(c));)
// plain add of an immediate (VIADD on sm_100)
KERNEL(k_viadd, asm volatile("add.u32 %0, %0, 0x1234567;" : "+r"(x[j]));)
// three-input add (IADD3)
KERNEL(k_iadd3, asm volatile("add.u32 %0, %0, %1;\n add.u32 %0, %0, %2;" : "+r"(x[j]) : "r"(b), "r"(c));)
// IMAD, all-register operands
KERNEL(k_imad_reg, asm volatile("mad.lo.u32 %0, %0, %1, %2;" : "+r"(x[j]) : "r"(b), "r"(c));)
// IMAD with an immediate multiplier
KERNEL(k_imad_imm, asm volatile("mad.lo.u32 %0, %0, 0x80002001, %1;" : "+r"(x[j]) : "r"(c));)
// LOP3 three-way xor
KERNEL(k_lop3, asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(x[j]) : "r"(b), "r"(c));)
// PRMT
KERNEL(k_prmt, asm volatile("prmt.b32 %0, %0, %1, 0x2104;" : "+r"(x[j]) : "r"(b));)
// FSETP + predicated FADD (float compare on the low bits' pattern)
KERNEL(k_fsetp, asm volatile("{\n .reg .pred p;\n setp.eq.f32 p, %0, %1;\n @p add.u32 %0, %0, 1;\n"
                             " mad.lo.u32 %0, %0, %2, %1;\n}" : "+r"(x[j]) : "r"(b), "r"(c));)

typedef void (*kfn)(uint32_t *, uint32_t, uint32_t, uint32_t);
int main() {
    uint32_t *out;
    cudaMalloc(&out, 4096);
    struct { const char *n; kfn f; int ops; } ks[] = {
        {"lop3p_viadd", k_lop3p_viadd, 3}, {"viadd", k_viadd, 1}, {"iadd3", k_iadd3, 2},
        {"imad_reg", k_imad_reg, 1}, {"imad_imm", k_imad_imm, 1}, {"lop3", k_lop3, 1},
        {"prmt", k_prmt, 1}, {"fsetp", k_fsetp, 3}};
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    int clk = 0;
    cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    for (auto &k : ks) {
        const int blocks = sms * 4, thr = 512;
        k.f<<<blocks, thr>>>(out, 1, 0x5bd1e995, 7);
        cudaEventRecord(e0);
        k.f<<<blocks, thr>>>(out, 1, 0x5bd1e995, 7);
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
        float ms = 0;
        cudaEventElapsedTime(&ms, e0, e1);
        const double lane_ops = (double)blocks * thr * IT * CH * k.ops;
        const double per_clk_sm = lane_ops / (ms * 1e-3) / (clk * 1e3) / sms;
        printf("%-12s %8.3f ms  %6.1f lane-instr/clk/SM (SASS instr per body as counted: %d)\n", k.n, ms,
               per_clk_sm, k.ops);
    }
    return cudaGetLastError() != cudaSuccess;
}

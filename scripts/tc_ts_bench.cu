// tc_ts_bench.cu -- microbenchmark (not product code): tcgen05 MMA issue rate with the A operand read from
// shared memory (SS, the production k_corr_tc scheme: Q rows share each A K-step) versus A copied once per
// K-step into tensor memory with tcgen05.cp and read from there by the Q row MMAs (TS).  Question: does
// moving A off the shared-memory port (128 -> ~85 B/clk/SM at Q = 3) raise the tensor-pipe rate?
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o tc_ts_bench scripts/tc_ts_bench.cu
// Each CTA (one per SM) runs ITERS K-steps; per K-step: [cp A] + Q x MMA(M=128, N=128, K=16) on
// distinct TMEM accumulator rows; commit every 4 K-steps to an mbarrier the issuing thread waits on
// every 8 K-steps (bounded queue).  Reports cycles per MMA.
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>

__device__ __forceinline__ uint32_t su32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }

__device__ __forceinline__ uint64_t desc(uint32_t saddr, uint32_t lbo, uint32_t sbo)
{
    uint64_t d = 0;
    d |= (uint64_t)((saddr >> 4) & 0x3FFF);
    d |= (uint64_t)((lbo >> 4) & 0x3FFF) << 16;
    d |= (uint64_t)((sbo >> 4) & 0x3FFF) << 32;
    d |= (uint64_t)1 << 46;
    return d;
}
__host__ __device__ constexpr uint32_t idesc(int m, int n)
{
    return (1u << 4) | (1u << 7) | (1u << 10) | ((uint32_t)(n >> 3) << 17) | ((uint32_t)(m >> 4) << 24);
}

template <int MODE, int Q>   // MODE 0 = SS, 1 = TS with cp, 2 = TS without cp (upper bound)
__global__ void __launch_bounds__(128, 1) bench(int iters, unsigned long long* out)
{
    extern __shared__ __align__(1024) unsigned char smem[];
    __shared__ uint64_t bar[2];
    __shared__ uint32_t tbase;
    const int warp = threadIdx.x >> 5;
    // A: 16 K-steps x 4 KB; B: Q rows + 4 x 2 KB... just one 16 KB region re-read
    for (int i = threadIdx.x; i < 96 * 1024 / 4; i += blockDim.x) reinterpret_cast<uint32_t*>(smem)[i] = 0x3c003c00u;
    if (threadIdx.x == 0) {
        asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(su32(&bar[0])), "r"(1));
        asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(su32(&bar[1])), "r"(1));
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == 0) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(su32(&tbase)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    asm volatile("tcgen05.fence::before_thread_sync;");
    __syncthreads();
    asm volatile("tcgen05.fence::after_thread_sync;");
    const uint32_t tmem = tbase;
    long long t0 = 0, t1 = 0;
    if (threadIdx.x == 0) {
        const uint32_t a0 = su32(smem), b0 = su32(smem + 64 * 1024);
        const uint64_t dA = desc(a0, 2048, 128), dB = desc(b0, 16, 128);
        constexpr uint32_t id = idesc(128, 128);
        const uint32_t acol = Q * 128;   // A ring in TMEM after the Q accumulator rows (TS)
        uint32_t phase[2] = {0, 0};
        t0 = clock64();
        for (int it = 0; it < iters; it++) {
            const int ks = it & 15;
            if (MODE == 1)
                asm volatile("tcgen05.cp.cta_group::1.128x256b [%0], %1;" ::"r"(tmem + acol + (ks & 15) * 8),
                             "l"(dA + ((ks * 4096) >> 4)));
#pragma unroll
            for (int q = 0; q < Q; q++) {
                const uint64_t db = dB + ((q * 2096 + (ks & 3) * 32) >> 4);
                if (MODE == 0) {
                    asm volatile("{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
                                 "tcgen05.mma.cta_group::1.kind::f16 [%0], %1, %2, %3, p;\n\t}\n" ::"r"(tmem + q * 128),
                                 "l"(dA + ((ks * 4096) >> 4)), "l"(db), "r"(id), "r"(1));
                } else {
                    asm volatile("{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
                                 "tcgen05.mma.cta_group::1.kind::f16 [%0], [%1], %2, %3, p;\n\t}\n" ::"r"(tmem + q * 128),
                                 "r"(tmem + acol + (ks & 15) * 8), "l"(db), "r"(id), "r"(1));
                }
            }
            if ((it & 7) == 7) {   // bound the queue: commit this period, wait for the previous one
                const int b = (it >> 3) & 1;
                asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(
                    su32(&bar[b])));
                if (it >= 15) {
                    uint32_t ok = 0;
                    while (!ok)
                        asm volatile("{\n\t.reg .pred p;\n\tmbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
                                     "selp.u32 %0, 1, 0, p;\n}\n"
                                     : "=r"(ok)
                                     : "r"(su32(&bar[b ^ 1])), "r"(phase[b ^ 1]));
                    phase[b ^ 1] ^= 1;
                }
            }
        }
        t1 = clock64();
        atomicAdd(out, (unsigned long long)(t1 - t0));
    }
    asm volatile("tcgen05.fence::before_thread_sync;");
    __syncthreads();
    if (warp == 0) asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
}

template <int MODE, int Q>
void run(const char* name)
{
    unsigned long long* d;
    cudaMalloc(&d, 8);
    cudaMemset(d, 0, 8);
    auto k = bench<MODE, Q>;
    cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, 100 * 1024);
    const int iters = 1 << 16;
    k<<<148, 128, 100 * 1024>>>(256, d);   // warm-up
    cudaDeviceSynchronize();
    cudaMemset(d, 0, 8);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    cudaEventRecord(e0);
    k<<<148, 128, 100 * 1024>>>(iters, d);
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms = 0;
    cudaEventElapsedTime(&ms, e0, e1);
    unsigned long long cyc = 0;
    cudaMemcpy(&cyc, d, 8, cudaMemcpyDeviceToHost);
    const double mmas = double(iters) * Q * 148;
    const double flop = mmas * 2.0 * 128 * 128 * 16;
    printf("%-28s Q=%d  %.2f cycles/MMA  %.1f TFLOP/s (bf16 dense executed)  err=%s\n", name, Q,
           double(cyc) / 148.0 / (double(iters) * Q), flop / (ms * 1e-3) / 1e12, cudaGetErrorString(cudaGetLastError()));
    cudaFree(d);
}

int main()
{
    run<0, 4>("SS (A from smem)");
    run<0, 3>("SS (A from smem)");
    run<1, 3>("TS + tcgen05.cp per K-step");
    run<2, 3>("TS, no copy (bound)");
    run<1, 2>("TS + tcgen05.cp per K-step");
    return 0;
}

// tc_issue_probe.cu -- probe (not product code): issue rate of tcgen05.mma (M=128, N=128, K=16, bf16, 4 TMEM
// accumulators) from one thread under three descriptor schemes, cycles per MMA:
//   0: every B descriptor an immediate offset (the dense unrolled schedule of k_corr_tc);
//   1: B offsets read from a shared-memory table per K-step (LDS -> R2UR -> MMA);
//   2: dense unrolled K-steps predicated by a runtime mask, A position from a running counter (skipped
//      K-steps issue nothing).
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/tc_issue_probe scripts/tc_issue_probe.cu
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>

__device__ __forceinline__ uint32_t su32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ uint64_t desc(uint32_t saddr, uint32_t lbo, uint32_t sbo)
{
    return (uint64_t)((saddr >> 4) & 0x3FFF) | ((uint64_t)((lbo >> 4) & 0x3FFF) << 16) |
           ((uint64_t)((sbo >> 4) & 0x3FFF) << 32) | ((uint64_t)1 << 46);
}
constexpr uint32_t IDESC = (1u << 4) | (1u << 7) | (1u << 10) | ((uint32_t)(128 >> 3) << 17) | ((uint32_t)(128 >> 4) << 24);
__device__ __forceinline__ void mma(uint32_t d, uint64_t a, uint64_t b, uint32_t acc)
{
    asm volatile("{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
                 "tcgen05.mma.cta_group::1.kind::f16 [%0], %1, %2, %3, p;\n\t}" ::"r"(d),
                 "l"(a), "l"(b), "r"(IDESC), "r"(acc)
                 : "memory");
}
__device__ __forceinline__ void mbar_init(uint64_t* b, int n)
{
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(su32(b)), "r"(n));
}
__device__ __forceinline__ void mbar_wait(uint64_t* b, uint32_t ph)
{
    asm volatile("{\n\t.reg .pred p;\n\tW: mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t@!p bra W;\n\t}" ::"r"(
                     su32(b)), "r"(ph)
                 : "memory");
}

constexpr int NS = 48;         // dense K-steps per tile
constexpr int ROWB = 2096;     // bytes per receptor row (131 x 16)
template <int MODE>
__global__ void __launch_bounds__(128, 1) probe(int tiles, unsigned long long mask, unsigned long long* cyc)
{
    extern __shared__ __align__(1024) unsigned char smem[];   // A ring 4 x 16 KB | B 58 KB
    __shared__ uint64_t bar;
    __shared__ uint32_t tbase;
    __shared__ __align__(16) uint16_t tab[NS];
    const int warp = threadIdx.x >> 5;
    for (int i = threadIdx.x; i < (64 * 1024 + 60 * 1024) / 16; i += blockDim.x)
        reinterpret_cast<uint4*>(smem)[i] = make_uint4(0, 0, 0, 0);
    if (threadIdx.x < NS) tab[threadIdx.x] = (uint16_t)((((threadIdx.x / 8) % 3) * 7 * ROWB + ((threadIdx.x / 2) % 4) * ROWB +
                                                          (threadIdx.x % 2) * 32) >> 4);
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    if (threadIdx.x == 0) {
        mbar_init(&bar, 1);
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
    long long t0 = clock64();
    int issued = 0;
    if (threadIdx.x == 0) {
        const uint32_t a0 = su32(smem), b0 = su32(smem + 64 * 1024);
        const uint64_t dA0 = desc(a0, 128 * 16, 128), dB0 = desc(b0, 16, 128);
        uint32_t apos = 0;   // A entry position in the 16-entry ring (4 stages x 4 K-steps)
        for (int t = 0; t < tiles; t++) {
            if (MODE == 0) {
#pragma unroll
                for (int s = 0; s < NS; s++) {
                    const uint64_t da = dA0 + (((s % 16) * 4096) >> 4);
                    const uint64_t db = dB0 + (((((s / 8) % 3) * 7 * ROWB + ((s / 2) % 4) * ROWB + (s % 2) * 32)) >> 4);
#pragma unroll
                    for (int q = 0; q < 4; q++) mma(tmem + q * 128, da, db + q * (ROWB >> 4), s ? 1u : 0u);
                }
                issued += NS * 4;
            } else if (MODE == 1) {
                for (int s0 = 0; s0 < NS; s0 += 4) {
                    const uint2 e2 = *reinterpret_cast<const uint2*>(tab + s0);
                    const uint32_t ev[4] = {e2.x & 0xffffu, e2.x >> 16, e2.y & 0xffffu, e2.y >> 16};
#pragma unroll
                    for (int k = 0; k < 4; k++) {
                        const uint64_t da = dA0 + ((((s0 + k) % 16) * 4096) >> 4);
                        const uint64_t db = dB0 + ev[k];
#pragma unroll
                        for (int q = 0; q < 4; q++) mma(tmem + q * 128, da, db + q * (ROWB >> 4), (s0 + k) ? 1u : 0u);
                    }
                }
                issued += NS * 4;
            } else {
#pragma unroll
                for (int s = 0; s < NS; s++) {
                    if ((mask >> s) & 1ull) {
                        const uint64_t da = dA0 + ((apos * 4096) >> 4);
                        apos = (apos + 1) & 15;
                        const uint64_t db = dB0 + (((((s / 8) % 3) * 7 * ROWB + ((s / 2) % 4) * ROWB + (s % 2) * 32)) >> 4);
#pragma unroll
                        for (int q = 0; q < 4; q++) mma(tmem + q * 128, da, db + q * (ROWB >> 4), 1u);
                    }
                }
                issued += __popcll(mask) * 4;
            }
        }
        asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(su32(&bar))
                     : "memory");
    }
    mbar_wait(&bar, 0);
    asm volatile("tcgen05.fence::after_thread_sync;");
    const long long t1 = clock64();
    if (threadIdx.x == 0) {
        cyc[2 * blockIdx.x] = (unsigned long long)(t1 - t0);
        cyc[2 * blockIdx.x + 1] = (unsigned long long)issued;
    }
    asm volatile("tcgen05.fence::before_thread_sync;");
    __syncthreads();
    if (warp == 0) asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
}

int main()
{
    const int blocks = 148, tiles = 200, smem = 64 * 1024 + 60 * 1024 + 1024;
    unsigned long long* dc;
    cudaMalloc(&dc, sizeof(unsigned long long) * 2 * blocks);
    unsigned long long hc[2 * 148];
    const unsigned long long masks[3] = {0xffffffffffffull, 0x5a5a5a5a5a5aull, 0x0f0f00f0f0f0ull};
    cudaFuncSetAttribute(probe<0>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    cudaFuncSetAttribute(probe<1>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    cudaFuncSetAttribute(probe<2>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    for (int mode = 0; mode < 3; mode++)
        for (int mi = 0; mi < (mode == 2 ? 3 : 1); mi++) {
            for (int rep = 0; rep < 2; rep++) {
                if (mode == 0) probe<0><<<blocks, 128, smem>>>(tiles, masks[mi], dc);
                if (mode == 1) probe<1><<<blocks, 128, smem>>>(tiles, masks[mi], dc);
                if (mode == 2) probe<2><<<blocks, 128, smem>>>(tiles, masks[mi], dc);
            }
            cudaError_t e = cudaDeviceSynchronize();
            cudaMemcpy(hc, dc, sizeof(hc), cudaMemcpyDeviceToHost);
            double mx = 0;
            for (int i = 0; i < blocks; i++) mx = hc[2 * i] > mx ? hc[2 * i] : mx;
            printf("mode %d mask %012llx %s: %.1f cycles per MMA (%llu MMAs)\n", mode, masks[mi],
                   e == cudaSuccess ? "ok" : cudaGetErrorString(e), mx / (double)hc[1], hc[1]);
        }
    return 0;
}

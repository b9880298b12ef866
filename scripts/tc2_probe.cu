// tc2_probe.cu -- probe (not product code) of the tcgen05 CTA-pair primitives the variant-3 correlation
// kernel needs, checked against a host reference and timed:
//   * tcgen05.alloc / dealloc .cta_group::2 (one warp in each CTA of the pair);
//   * tcgen05.mma.cta_group::2.kind::f16, M = 256 (A: 128 rows from each CTA's shared memory), N = 128
//     (B: 64 rows from each CTA), D: each CTA's TMEM holds its 128 rows x 128 columns;
//   * tcgen05.commit.cta_group::2 ... multicast::cluster (completion signalled in both CTAs);
//   * remote mbarrier arrive (mapa + mbarrier.arrive.release.cluster.shared::cluster).
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/tc2_probe scripts/tc2_probe.cu && /tmp/tc2_probe
#include <cuda_bf16.h>
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>

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
__device__ __forceinline__ uint32_t cta_rank()
{
    uint32_t r;
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
    return r;
}
__device__ __forceinline__ void cluster_sync()
{
    asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}
__device__ __forceinline__ void mbar_init(uint64_t* b, int n)
{
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(su32(b)), "r"(n));
}
__device__ __forceinline__ void mbar_wait(uint64_t* b, uint32_t ph)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\tW: mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t@!p bra W;\n\t}" ::"r"(su32(b)),
        "r"(ph)
        : "memory");
}
__device__ __forceinline__ void mbar_arrive_remote(uint64_t* local_b, uint32_t target_cta)
{
    uint32_t ra;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(ra) : "r"(su32(local_b)), "r"(target_cta));
    asm volatile("mbarrier.arrive.release.cluster.shared::cluster.b64 _, [%0];" ::"r"(ra) : "memory");
}

template <int CG>   // CG = 1: M = 128 per CTA (reference timing), 2: CTA pair, M = 256
__global__ void __cluster_dims__(2, 1, 1) __launch_bounds__(128, 1) probe(const uint16_t* __restrict__ A,
                                                                            const uint16_t* __restrict__ B, int ksteps,
                                                                            int reps, float* D, unsigned long long* cyc)
{
    // A: per CTA [ks][2 chunks][128 rows][8 bf16]; B: per CTA its half [ks][2][64][8] (CG = 2) or all [ks][2][128][8]
    extern __shared__ __align__(1024) unsigned char smem[];
    __shared__ uint64_t bar_done, bar_peer;
    __shared__ uint32_t tbase;
    const uint32_t rank = cta_rank();
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int nB = CG == 2 ? 64 : 128;
    const size_t a_bytes = (size_t)ksteps * 2 * 128 * 16, b_bytes = (size_t)ksteps * 2 * nB * 16;
    {
        const uint4* As = reinterpret_cast<const uint4*>(A + (size_t)rank * ksteps * 2 * 128 * 8);
        const uint4* Bs = reinterpret_cast<const uint4*>(B + (CG == 2 ? (size_t)rank * ksteps * 2 * 64 * 8 : 0));
        uint4* sa = reinterpret_cast<uint4*>(smem);
        uint4* sb = reinterpret_cast<uint4*>(smem + a_bytes);
        for (size_t i = threadIdx.x; i < a_bytes / 16; i += blockDim.x) sa[i] = As[i];
        for (size_t i = threadIdx.x; i < b_bytes / 16; i += blockDim.x) sb[i] = Bs[i];
    }
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");   // generic-proxy writes -> async proxy (MMA)
    if (threadIdx.x == 0) {
        mbar_init(&bar_done, 1);
        mbar_init(&bar_peer, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == 0) {
        if (CG == 2) {
            asm volatile("tcgen05.alloc.cta_group::2.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(su32(&tbase)));
            asm volatile("tcgen05.relinquish_alloc_permit.cta_group::2.sync.aligned;");
        } else {
            asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(su32(&tbase)));
            asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
        }
    }
    asm volatile("tcgen05.fence::before_thread_sync;");
    __syncthreads();
    cluster_sync();
    asm volatile("tcgen05.fence::after_thread_sync;");
    const uint32_t tmem = tbase;
    // peer handshake through a remote arrive: rank 1 -> rank 0
    if (CG == 2 && rank == 1 && threadIdx.x == 0) mbar_arrive_remote(&bar_peer, 0);
    if (CG == 2 && rank == 0 && threadIdx.x == 0) mbar_wait(&bar_peer, 0);
    const bool issuer = (CG == 1 || rank == 0) && threadIdx.x == 0;
    long long t0 = clock64();
    if (issuer) {
        const uint32_t a0 = su32(smem), b0 = su32(smem + a_bytes);
        constexpr uint32_t id = idesc(CG == 2 ? 256 : 128, 128);
        // Q = 4 independent accumulators (TMEM columns q * 128) interleaved per K-step, as in k_corr_tc
        for (int rep = 0; rep < reps; rep++) {
            for (int ks = 0; ks < ksteps; ks++) {
                const uint64_t dA = desc(a0 + ks * 2 * 128 * 16, 128 * 16, 128);
                const uint64_t dB = desc(b0 + ks * 2 * nB * 16, nB * 16, 128);
                const uint32_t acc = (rep > 0 || ks > 0) ? 1u : 0u;
#pragma unroll
                for (int q = 0; q < 4; q++) {
                    const uint32_t dcol = tmem + (uint32_t)q * 128u;
                    if (CG == 2)
                        asm volatile(
                            "{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
                            "tcgen05.mma.cta_group::2.kind::f16 [%0], %1, %2, %3, p;\n\t}" ::"r"(dcol),
                            "l"(dA), "l"(dB), "r"(id), "r"(acc)
                            : "memory");
                    else
                        asm volatile(
                            "{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
                            "tcgen05.mma.cta_group::1.kind::f16 [%0], %1, %2, %3, p;\n\t}" ::"r"(dcol),
                            "l"(dA), "l"(dB), "r"(id), "r"(acc)
                            : "memory");
                }
            }
        }
        if (CG == 2)
            asm volatile(
                "tcgen05.commit.cta_group::2.mbarrier::arrive::one.shared::cluster.multicast::cluster.b64 [%0], %1;" ::"r"(
                    su32(&bar_done)),
                "h"((uint16_t)3)
                : "memory");
        else
            asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(
                su32(&bar_done))
                         : "memory");
    }
    mbar_wait(&bar_done, 0);
    asm volatile("tcgen05.fence::after_thread_sync;");
    const long long t1 = clock64();
    if (threadIdx.x == 0) cyc[blockIdx.x] = (unsigned long long)(t1 - t0);
    // D: TMEM lane = row of this CTA's 128, column = n
    for (int c0 = 0; c0 < 128; c0 += 32) {
        uint32_t v[32];
        const uint32_t addr = tmem + ((uint32_t)(warp * 32) << 16) + c0;
        asm volatile(
            "tcgen05.ld.sync.aligned.32x32b.x32.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,%16,%17,%18,%"
            "19,%20,%21,%22,%23,%24,%25,%26,%27,%28,%29,%30,%31}, [%32];"
            : "=r"(v[0]), "=r"(v[1]), "=r"(v[2]), "=r"(v[3]), "=r"(v[4]), "=r"(v[5]), "=r"(v[6]), "=r"(v[7]), "=r"(v[8]),
              "=r"(v[9]), "=r"(v[10]), "=r"(v[11]), "=r"(v[12]), "=r"(v[13]), "=r"(v[14]), "=r"(v[15]), "=r"(v[16]),
              "=r"(v[17]), "=r"(v[18]), "=r"(v[19]), "=r"(v[20]), "=r"(v[21]), "=r"(v[22]), "=r"(v[23]), "=r"(v[24]),
              "=r"(v[25]), "=r"(v[26]), "=r"(v[27]), "=r"(v[28]), "=r"(v[29]), "=r"(v[30]), "=r"(v[31])
            : "r"(addr));
        asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
        const int row = warp * 32 + lane;
        for (int j = 0; j < 32; j++)
            D[((size_t)blockIdx.x * 128 + row) * 128 + c0 + j] = __uint_as_float(v[j]);
    }
    asm volatile("tcgen05.fence::before_thread_sync;");
    __syncthreads();
    cluster_sync();
    if (warp == 0) {
        if (CG == 2)
            asm volatile("tcgen05.dealloc.cta_group::2.sync.aligned.b32 %0, 512;" ::"r"(tmem));
        else
            asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
    }
}

static uint16_t bf(float x)
{
    __nv_bfloat16 h = __float2bfloat16(x);
    return *reinterpret_cast<uint16_t*>(&h);
}

int main()
{
    const int ks = 8, pairs = 74;
    const int reps_check = 1, reps_time = 100;
    // logical A_c [128 rows][16 ks elements], per CTA c of each pair; B [128 n][16 ks]
    const size_t nA = (size_t)2 * ks * 2 * 128 * 8, nB = (size_t)ks * 2 * 128 * 8;
    uint16_t *hA = (uint16_t*)malloc(nA * 2), *hB = (uint16_t*)malloc(nB * 2), *hB2 = (uint16_t*)malloc(nB * 2);
    float* Al = (float*)malloc(sizeof(float) * 2 * 128 * ks * 16);
    float* Bl = (float*)malloc(sizeof(float) * 128 * ks * 16);
    srand(7);
    for (int c = 0; c < 2; c++)
        for (int r = 0; r < 128; r++)
            for (int k = 0; k < ks * 16; k++) {
                const float v = (float)(rand() % 9 - 4);
                Al[((size_t)c * 128 + r) * ks * 16 + k] = v;
                const int s = k / 16, kk = k % 16, ch = kk / 8, e = kk % 8;
                hA[(size_t)c * ks * 2 * 128 * 8 + (((size_t)s * 2 + ch) * 128 + r) * 8 + e] = bf(v);
            }
    for (int n = 0; n < 128; n++)
        for (int k = 0; k < ks * 16; k++) {
            const float v = (float)(rand() % 7 - 3);
            Bl[(size_t)n * ks * 16 + k] = v;
            const int s = k / 16, kk = k % 16, ch = kk / 8, e = kk % 8;
            // CG = 1 layout: [s][ch][128][8]; CG = 2: CTA half h = n / 64: [h][s][ch][64][8]
            hB[(((size_t)s * 2 + ch) * 128 + n) * 8 + e] = bf(v);
            const int h = n / 64, nn = n % 64;
            hB2[(size_t)h * ks * 2 * 64 * 8 + (((size_t)s * 2 + ch) * 64 + nn) * 8 + e] = bf(v);
        }
    uint16_t *dA, *dB, *dB2;
    float* dD;
    unsigned long long* dc;
    cudaMalloc(&dA, nA * 2);
    cudaMalloc(&dB, nB * 2);
    cudaMalloc(&dB2, nB * 2);
    cudaMalloc(&dD, sizeof(float) * 2 * pairs * 128 * 128);
    cudaMalloc(&dc, sizeof(unsigned long long) * 2 * pairs);
    cudaMemcpy(dA, hA, nA * 2, cudaMemcpyHostToDevice);
    cudaMemcpy(dB, hB, nB * 2, cudaMemcpyHostToDevice);
    cudaMemcpy(dB2, hB2, nB * 2, cudaMemcpyHostToDevice);
    const int smem = (int)(nA / 2 * 2 + nB * 2) + 1024;
    cudaFuncSetAttribute(probe<1>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    cudaFuncSetAttribute(probe<2>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    float* hD = (float*)malloc(sizeof(float) * 2 * pairs * 128 * 128);
    unsigned long long hc[2 * 74];
    for (int cg = 1; cg <= 2; cg++) {
        // correctness (1 rep)
        if (cg == 1)
            probe<1><<<2 * pairs, 128, smem>>>(dA, dB, ks, reps_check, dD, dc);
        else
            probe<2><<<2 * pairs, 128, smem>>>(dA, dB2, ks, reps_check, dD, dc);
        cudaError_t e = cudaDeviceSynchronize();
        if (e != cudaSuccess) {
            printf("cg=%d launch error: %s\n", cg, cudaGetErrorString(e));
            return 1;
        }
        cudaMemcpy(hD, dD, sizeof(float) * 2 * 128 * 128, cudaMemcpyDeviceToHost);
        double maxerr = 0;
        for (int c = 0; c < 2; c++)
            for (int r = 0; r < 128; r++)
                for (int n = 0; n < 128; n++) {
                    // CG = 1: every CTA uses A of its rank-in-pair (blockIdx % 2) and the full B
                    double ref = 0;
                    for (int k = 0; k < ks * 16; k++)
                        ref += (double)Al[((size_t)c * 128 + r) * ks * 16 + k] * Bl[(size_t)n * ks * 16 + k];
                    const double got = hD[((size_t)c * 128 + r) * 128 + n];
                    if (fabs(got - ref) > maxerr) maxerr = fabs(got - ref);
                }
        // timing
        if (cg == 1)
            probe<1><<<2 * pairs, 128, smem>>>(dA, dB, ks, reps_time, dD, dc);
        else
            probe<2><<<2 * pairs, 128, smem>>>(dA, dB2, ks, reps_time, dD, dc);
        e = cudaDeviceSynchronize();
        cudaMemcpy(hc, dc, sizeof(hc), cudaMemcpyDeviceToHost);
        double mx = 0;
        for (int i = 0; i < 2 * pairs; i++) mx = hc[i] > mx ? hc[i] : mx;
        const double n_mma = (double)reps_time * ks * 4;   // instructions issued per issuing CTA
        const double per_sm_128 = mx / n_mma;   // each SM's share of one instruction is 128x128x16 in both modes
        printf("cg=%d %s max|err| %.3g  cycles per instruction %.1f = cycles per 128x128x16 MACs per SM "
               "(nominal 2.25 PF at 1965 MHz: 67.8)\n", cg, e == cudaSuccess ? "ok" : cudaGetErrorString(e), maxerr,
               per_sm_128);
    }
    return 0;
}

// tc_proto2.cu -- swapped-role variant (A = weights, M = 128 rotations; B = receptor rows,
// N = 128 translations) of the standalone feasibility test of the tcgen05 implicit-GEMM form of the
// multi-term direct correlation.  Not part of libdock.so.
//
// C[t][r] = sum_{v, p} R_p(t + v) * W_r(v, p), computed as bf16x3 on the tensor cores:
//   A (M = 128 consecutive x translations, K-major) is read straight out of a receptor tile
//   stored [z][y][x][8 bf16] with the 8 "channels" = (hi_0..3, lo_0..3): a filter offset v is
//   only a descriptor start-address offset (rows 16 B apart, core-matrix groups SBO = 128 B,
//   the two K-chunks of one K=16 MMA = voxels vx and vx+1, LBO = 16 B).
//   B (N rotations, K-major): pass 1 chunk = (Whi_0..3, Whi_0..3) -> Rhi*Whi + Rlo*Whi,
//                             pass 2 chunk = (Wlo_0..3, 0..0)    -> Rhi*Wlo.
// Output compared with an FP64 host reference; prints max err / A.
#include <cuda_bf16.h>
#include <cuda_runtime.h>

#include <cmath>
#include <cstdint>
#include <cstdio>
#include <cstdlib>
#include <vector>

constexpr int M = 2;            // probe grid edge
constexpr int P = 4;            // channels
constexpr int NX = 128, NY = 2, NZ = 2;
constexpr int TXB = 136;        // 128 + M - 1 -> padded
constexpr int TYB = NY + M - 1, TZB = NZ + M - 1;
constexpr int NROT = 128;       // MMA M (rotations)
constexpr int NSTEP = 2 * M * M * (M / 2);   // passes x vz x vy x vx-pairs = 64
constexpr int NQ = NY * NZ;     // M-blocks (rows of 128 translations)

__host__ __device__ inline uint32_t smem_u32(const void* p)
{
#ifdef __CUDA_ARCH__
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
#else
    return 0;
#endif
}

__device__ __forceinline__ uint64_t make_desc(uint32_t saddr, uint32_t lbo, uint32_t sbo)
{
    uint64_t d = 0;
    d |= (uint64_t)((saddr >> 4) & 0x3FFF);
    d |= (uint64_t)((lbo >> 4) & 0x3FFF) << 16;
    d |= (uint64_t)((sbo >> 4) & 0x3FFF) << 32;
    d |= (uint64_t)1 << 46;   // version = 1 (sm100)
    // base_offset = 0, lbo_mode = 0, layout_type = 0 (SWIZZLE_NONE)
    return d;
}

__device__ __forceinline__ uint32_t make_idesc(int m, int n)
{
    uint32_t d = 0;
    d |= 1u << 4;          // c_format = F32
    d |= 1u << 7;          // a_format = BF16
    d |= 1u << 10;         // b_format = BF16
    d |= (uint32_t)(n >> 3) << 17;
    d |= (uint32_t)(m >> 4) << 24;
    return d;
}

__global__ void __launch_bounds__(128, 1) k_tc(const uint4* __restrict__ gA, const uint4* __restrict__ gB,
                                                float* __restrict__ out)
{
    extern __shared__ __align__(1024) unsigned char smem[];
    uint4* sA = reinterpret_cast<uint4*>(smem);                               // [TZB][TYB][TXB] x 16 B
    uint4* sB = reinterpret_cast<uint4*>(smem + TZB * TYB * TXB * 16);        // [NSTEP][2][NROT] x 16 B
    __shared__ uint64_t mbar;
    __shared__ uint32_t tmem_base;
    const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;

    for (int i = tid; i < TZB * TYB * TXB; i += blockDim.x) sA[i] = gA[i];
    for (int i = tid; i < NSTEP * 2 * NROT; i += blockDim.x) sB[i] = gB[i];
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
    if (warp == 0) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(smem_u32(&tmem_base)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    if (tid == 0) {
        asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(smem_u32(&mbar)));
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory");
    __syncthreads();
    asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory");
    const uint32_t tmem = tmem_base;

    if (tid == 0) {
        const uint32_t idesc = make_idesc(NROT, 128);
        const uint32_t a0 = smem_u32(sA), b0 = smem_u32(sB);
        for (int q = 0; q < NQ; q++) {
            const int y = q % NY, z = q / NY;
            for (int s = 0; s < NSTEP; s++) {
                const int vxp = s % (M / 2), vy = (s / (M / 2)) % M, vz = (s / (M / 2 * M)) % M;
                const uint32_t aoff = (((z + vz) * TYB + (y + vy)) * TXB + 2 * vxp) * 16;
                const uint64_t db = make_desc(a0 + aoff, 16, 128);                    // receptor rows = B (N)
                const uint64_t da = make_desc(b0 + s * 2 * NROT * 16, NROT * 16, 128);  // weights = A (M)
                const uint32_t dt = tmem + q * 128;
                const uint32_t acc = s > 0 ? 1u : 0u;
                asm volatile(
                    "{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
                    "tcgen05.mma.cta_group::1.kind::f16 [%0], %1, %2, %3, p;\n\t}\n" ::"r"(dt),
                    "l"(da), "l"(db), "r"(idesc), "r"(acc));
            }
        }
        asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(
                         smem_u32(&mbar))
                     : "memory");
    }
    // wait for all MMAs
    {
        uint32_t ok = 0;
        while (!ok) {
            asm volatile(
                "{\n\t.reg .pred p;\n\tmbarrier.try_wait.parity.shared::cta.b64 p, [%1], 0;\n\t"
                "selp.u32 %0, 1, 0, p;\n\t}\n"
                : "=r"(ok)
                : "r"(smem_u32(&mbar))
                : "memory");
        }
    }
    asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory");
    for (int q = 0; q < NQ; q++) {
        for (int c0 = 0; c0 < 128; c0 += 32) {
            uint32_t v[32];
            const uint32_t addr = tmem + ((uint32_t)(warp * 32) << 16) + q * 128 + c0;
            asm volatile(
                "tcgen05.ld.sync.aligned.32x32b.x32.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,"
                "%16,%17,%18,%19,%20,%21,%22,%23,%24,%25,%26,%27,%28,%29,%30,%31}, [%32];"
                : "=r"(v[0]), "=r"(v[1]), "=r"(v[2]), "=r"(v[3]), "=r"(v[4]), "=r"(v[5]), "=r"(v[6]), "=r"(v[7]),
                  "=r"(v[8]), "=r"(v[9]), "=r"(v[10]), "=r"(v[11]), "=r"(v[12]), "=r"(v[13]), "=r"(v[14]),
                  "=r"(v[15]), "=r"(v[16]), "=r"(v[17]), "=r"(v[18]), "=r"(v[19]), "=r"(v[20]), "=r"(v[21]),
                  "=r"(v[22]), "=r"(v[23]), "=r"(v[24]), "=r"(v[25]), "=r"(v[26]), "=r"(v[27]), "=r"(v[28]),
                  "=r"(v[29]), "=r"(v[30]), "=r"(v[31])
                : "r"(addr));
            asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
            const int r = warp * 32 + lane;   // TMEM lane = M row = rotation
            for (int j = 0; j < 32; j++) out[(size_t)(q * NX + c0 + j) * NROT + r] = __uint_as_float(v[j]);
        }
    }
    asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory");
    __syncthreads();
    if (warp == 0) asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
}

static uint16_t bf16_bits(float f)
{
    __nv_bfloat16 h = __float2bfloat16_rn(f);
    return *reinterpret_cast<uint16_t*>(&h);
}
static float bf16_val(uint16_t b)
{
    uint32_t u = (uint32_t)b << 16;
    float f;
    memcpy(&f, &u, 4);
    return f;
}

int main()
{
    srand(7);
    auto rnd = [] { return (float)rand() / RAND_MAX * 2.f - 1.f; };
    std::vector<float> R((size_t)P * NZ * NY * NX);
    for (auto& x : R) x = rnd() * 3.f;
    std::vector<float> W((size_t)NROT * P * M * M * M, 0.f);     // [r][p][vz][vy][vx]
    for (int r = 0; r < NROT; r++)
        for (int a = 0; a < 6; a++) {
            int v = rand() % (M * M * M);
            for (int p = 0; p < P; p++) W[((size_t)r * P + p) * M * M * M + v] += rnd();
        }
    // A tile: [TZB][TYB][TXB][8] bf16 (cyclic padding)
    std::vector<uint16_t> hA((size_t)TZB * TYB * TXB * 8, 0);
    for (int z = 0; z < TZB; z++)
        for (int y = 0; y < TYB; y++)
            for (int x = 0; x < TXB; x++)
                for (int p = 0; p < P; p++) {
                    float f = R[(((size_t)p * NZ + z % NZ) * NY + y % NY) * NX + x % NX];
                    uint16_t hi = bf16_bits(f);
                    uint16_t lo = bf16_bits(f - bf16_val(hi));
                    size_t o = (((size_t)z * TYB + y) * TXB + x) * 8;
                    hA[o + p] = hi;
                    hA[o + 4 + p] = lo;
                }
    // B: [step][chunk][rot][8]
    std::vector<uint16_t> hB((size_t)NSTEP * 2 * NROT * 8, 0);
    for (int s = 0; s < NSTEP; s++) {
        const int vxp = s % (M / 2), vy = (s / (M / 2)) % M, vz = (s / (M / 2 * M)) % M, pass = s / (M / 2 * M * M);
        for (int c = 0; c < 2; c++)
            for (int r = 0; r < NROT; r++)
                for (int p = 0; p < P; p++) {
                    int vx = 2 * vxp + c;
                    float f = W[((size_t)r * P + p) * M * M * M + (vz * M + vy) * M + vx];
                    uint16_t hi = bf16_bits(f), lo = bf16_bits(f - bf16_val(hi));
                    size_t o = (((size_t)s * 2 + c) * NROT + r) * 8;
                    if (pass == 0) {
                        hB[o + p] = hi;
                        hB[o + 4 + p] = hi;
                    } else {
                        hB[o + p] = lo;
                        hB[o + 4 + p] = 0;
                    }
                }
    }
    uint4 *dA, *dB;
    float* dO;
    cudaMalloc(&dA, hA.size() * 2);
    cudaMalloc(&dB, hB.size() * 2);
    cudaMalloc(&dO, sizeof(float) * NQ * NX * NROT);
    cudaMemcpy(dA, hA.data(), hA.size() * 2, cudaMemcpyHostToDevice);
    cudaMemcpy(dB, hB.data(), hB.size() * 2, cudaMemcpyHostToDevice);
    size_t smem = (size_t)TZB * TYB * TXB * 16 + (size_t)NSTEP * 2 * NROT * 16;
    cudaFuncSetAttribute(k_tc, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    k_tc<<<1, 128, smem>>>(dA, dB, dO);
    cudaError_t e = cudaDeviceSynchronize();
    printf("kernel: %s (smem %zu)\n", cudaGetErrorString(e), smem);
    std::vector<float> O((size_t)NQ * NX * NROT);
    cudaMemcpy(O.data(), dO, O.size() * 4, cudaMemcpyDeviceToHost);
    double maxerr = 0, maxrel = 0;
    for (int q = 0; q < NQ; q++)
        for (int x = 0; x < NX; x++)
            for (int r = 0; r < NROT; r++) {
                int y = q % NY, z = q / NY;
                double s = 0, a = 0;
                for (int p = 0; p < P; p++)
                    for (int vz = 0; vz < M; vz++)
                        for (int vy = 0; vy < M; vy++)
                            for (int vx = 0; vx < M; vx++) {
                                double w = W[((size_t)r * P + p) * M * M * M + (vz * M + vy) * M + vx];
                                double rv = R[(((size_t)p * NZ + (z + vz) % NZ) * NY + (y + vy) % NY) * NX +
                                              (x + vx) % NX];
                                s += w * rv;
                                a += fabs(w * rv);
                            }
                double g = O[((size_t)q * NX + x) * NROT + r];
                maxerr = fmax(maxerr, fabs(g - s));
                if (a > 0) maxrel = fmax(maxrel, fabs(g - s) / a);
            }
    printf("max |err| = %.3e   max err/A = %.3e  -> %s\n", maxerr, maxrel, maxrel < 1e-4 ? "PASS" : "FAIL");
    return maxrel < 1e-4 ? 0 : 1;
}

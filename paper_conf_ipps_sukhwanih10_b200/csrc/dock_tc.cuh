// dock_tc.cuh -- tensor-core (tcgen05) engine of the multi-term direct correlation
// (north star (b): "Tensor cores are used only if an implicit-GEMM
// form over the term channels meets the stated tolerance").
//
// Implicit GEMM per (rotation block, translation row):
//   D[r][x] = sum_K A[r][K] * B[x][K],   r = 128 rotations (MMA M), x = 128 translations
//   along one receptor x-row (MMA N), K = (channel group g, pass, vz, vy, vx, 8 "channels").
// bf16x3 split keeps FP32-level accuracy (|err| ~ 1e-5 * A, tolerance 1e-4 * A, reading Q16):
//   receptor voxel = 8 bf16 (Rhi_0..3, Rlo_0..3) of 4 channels, 16 B;
//   pass 0 weights = (Whi_0..3, Whi_0..3)  -> Rhi*Whi + Rlo*Whi,
//   pass 1 weights = (Wlo_0..3, 0, 0, 0, 0) -> Rhi*Wlo.
// B needs no im2col: the receptor tile is stored [z][y][x][8 bf16] in shared memory, so the
// K-major no-swizzle UMMA layout (core matrix = 8 rows x 16 B, rows 16 B apart, SBO = 128 B)
// of "128 consecutive translations x (voxel vx, vx+1)" is the tile itself read at a start
// address offset of the filter offset (vz, vy, vx); LBO = 16 B steps to voxel vx+1.
// A (weights, K-major) streams through an 8-stage mbarrier ring (4 KB per K-step) and is
// reused by the Q translation rows of a tile; D lives in TMEM (Q x 128 columns per buffer).
// Epilogue: one thread per (rotation, half of the rows) reads its TMEM lane with
// tcgen05.ld and keeps an exact per-thread top-LIST key list (no score grid in HBM),
// published at item end exactly like the FFMA engine (k_merge is shared).
#pragma once
#include <cuda_bf16.h>

#include "dock_kernels.cuh"

namespace tc {

using dk::KEY_MAX;

constexpr int ROT = 128;        // rotations per block (MMA M)
constexpr int NT = 128;         // translations per row (MMA N)
constexpr int NEPI_MAX = 16;    // epilogue warps: a.nepi in {4, 8, 16} (1, 2 or 4 per TMEM lane quarter)
constexpr int NTHREADS = (2 + NEPI_MAX) * 32;   // launch bound; the launch uses (2 + a.nepi) * 32 threads
constexpr int WSTAGES = 16;     // max weight ring depth (runtime a.wstages <= 16; 16 x 4 KB covers the L2 latency)
constexpr int WCHUNK = 2 * ROT * 16;   // bytes of one K-step of A (2 K-chunks x 128 rotations x 16 B)
constexpr int KSTEPS = 4;       // K-steps of A per ring stage (one elected issue block of KSTEPS*Q MMAs)
constexpr int LIST = 16;        // per-thread candidate list (exact top-LIST keys of one rotation and row class)

struct TcArgs {
    int nx, ny, nz;
    int ntx, nty, ntz, ntiles;  // tiles: 128 x Q rows (y) x 1 (z)
    int G_ch;                   // channel groups of 4
    int n_slots, G, tiles_per_region;
    int nsteps;                 // K-steps of A per tile (all passes, padded to multiples of KSTEPS)
    int S1, S1p, S2, S2p;       // PAIR scheme: pass-1 steps (real, padded) and pass-2 steps (real, padded)
    const unsigned char* W;     // [block][step][WCHUNK]
    int TXB, TYB, TZB;
    int box_bytes;              // one channel group's receptor box
    int rec_stage_bytes;        // G_ch * box_bytes rounded to 1024
    int n_rec_stages;           // 1 or 2
    int wstages;                // weight ring depth (3..WSTAGES)
    int nepi;                   // epilogue warps (4, 8 or 16)
    // top-k
    int k, rho, cap;
    unsigned long long* T;
    unsigned long long* mu;
    unsigned int* cnt;
    unsigned long long* cand;
    // grid mode
    float* grid;
    // diagnostics (DOCK_TC_TRACE / DOCK_TC_DEBUG environment variables; off on the product path):
    // trace = per-role cycle counters summed over CTAs (see TR_*); dbg 1 = epilogue skips the TMEM
    // drain, 2 = drain without candidate processing (timing experiments only: poses are invalid)
    unsigned long long* trace;
    int dbg;
};

// trace counters (cycles summed over CTAs)
enum { TR_CTAS = 0, TR_TILES, TR_MMA_TOTAL, TR_MMA_TMEMPTY, TR_MMA_WFULL, TR_MMA_RFULL, TR_EPI_TOTAL, TR_EPI_TMFULL,
       TR_EPI_LDTM, TR_PROD_TOTAL, TR_PROD_WEMPTY, TR_PROD_REMPTY, TR_EPI_WARPS, TR_N = 16 };

// mbarrier wait that adds its duration to `acc` when tracing
__device__ __forceinline__ void twait(uint64_t* bar, unsigned parity, bool tr, long long& acc)
{
    if (tr) {
        const long long t0 = clock64();
        dk::mbar_wait(bar, parity);
        acc += clock64() - t0;
    } else {
        dk::mbar_wait(bar, parity);
    }
}

__device__ __forceinline__ uint64_t umma_desc(uint32_t saddr, uint32_t lbo, uint32_t sbo)
{
    uint64_t d = 0;
    d |= static_cast<uint64_t>((saddr >> 4) & 0x3FFFu);
    d |= static_cast<uint64_t>((lbo >> 4) & 0x3FFFu) << 16;
    d |= static_cast<uint64_t>((sbo >> 4) & 0x3FFFu) << 32;
    d |= static_cast<uint64_t>(1) << 46;   // descriptor version 1 (sm_100); no swizzle, base offset 0
    return d;
}

// kind::f16 instruction descriptor: D f32, A/B bf16, both K-major, M x N.
__host__ __device__ constexpr uint32_t umma_idesc(int m, int n)
{
    return (1u << 4) | (1u << 7) | (1u << 10) | (static_cast<uint32_t>(n >> 3) << 17) |
           (static_cast<uint32_t>(m >> 4) << 24);
}

__device__ __forceinline__ void umma_bf16(uint32_t d_tmem, uint64_t a, uint64_t b, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::1.kind::f16 [%0], %1, %2, %3, p;\n\t}\n" ::"r"(d_tmem),
        "l"(a), "l"(b), "r"(idesc), "r"(acc)
        : "memory");
}
__device__ __forceinline__ void umma_commit(uint64_t* bar)
{
    asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(
                     dk::smem_u32(bar))
                 : "memory");
}
__device__ __forceinline__ void tc_fence_after() { asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory"); }
__device__ __forceinline__ void tc_fence_before() { asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory"); }

__device__ __forceinline__ void tmem_ld32(uint32_t addr, uint32_t (&v)[32])
{
    asm volatile(
        "tcgen05.ld.sync.aligned.32x32b.x32.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,"
        "%16,%17,%18,%19,%20,%21,%22,%23,%24,%25,%26,%27,%28,%29,%30,%31}, [%32];"
        : "=r"(v[0]), "=r"(v[1]), "=r"(v[2]), "=r"(v[3]), "=r"(v[4]), "=r"(v[5]), "=r"(v[6]), "=r"(v[7]),
          "=r"(v[8]), "=r"(v[9]), "=r"(v[10]), "=r"(v[11]), "=r"(v[12]), "=r"(v[13]), "=r"(v[14]), "=r"(v[15]),
          "=r"(v[16]), "=r"(v[17]), "=r"(v[18]), "=r"(v[19]), "=r"(v[20]), "=r"(v[21]), "=r"(v[22]),
          "=r"(v[23]), "=r"(v[24]), "=r"(v[25]), "=r"(v[26]), "=r"(v[27]), "=r"(v[28]), "=r"(v[29]),
          "=r"(v[30]), "=r"(v[31])
        : "r"(addr));
    asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
}

__device__ __forceinline__ void tma_load_5d(void* dst, const CUtensorMap* map, int c0, int c1, int c2, int c3,
                                            int c4, uint64_t* bar)
{
    asm volatile(
        "cp.async.bulk.tensor.5d.shared::cluster.global.tile.mbarrier::complete_tx::bytes"
        " [%0], [%1, {%2, %3, %4, %5, %6}], [%7];" ::"r"(dk::smem_u32(dst)),
        "l"(reinterpret_cast<uint64_t>(map)), "r"(c0), "r"(c1), "r"(c2), "r"(c3), "r"(c4),
        "r"(dk::smem_u32(bar))
        : "memory");
}

__device__ __forceinline__ bool elect_one()
{
    uint32_t pred = 0;
    asm volatile(
        "{\n\t.reg .pred P;\n\telect.sync _|P, 0xffffffff;\n\tselp.u32 %0, 1, 0, P;\n\t}\n"
        : "=r"(pred));
    return pred != 0;
}

// v[j] for a runtime j without local memory: binary select tree over the 5 bits of j.
__device__ __forceinline__ uint32_t select32(const uint32_t (&v)[32], int j)
{
    uint32_t l1[16], l2[8], l3[4], l4[2];
#pragma unroll
    for (int i = 0; i < 16; i++) l1[i] = (j & 1) ? v[2 * i + 1] : v[2 * i];
#pragma unroll
    for (int i = 0; i < 8; i++) l2[i] = (j & 2) ? l1[2 * i + 1] : l1[2 * i];
#pragma unroll
    for (int i = 0; i < 4; i++) l3[i] = (j & 4) ? l2[2 * i + 1] : l2[2 * i];
#pragma unroll
    for (int i = 0; i < 2; i++) l4[i] = (j & 8) ? l3[2 * i + 1] : l3[2 * i];
    return (j & 16) ? l4[1] : l4[0];
}

// Sorted (ascending) per-thread key list, fully unrolled insertion.
__device__ __forceinline__ void list_insert(unsigned long long (&L)[LIST], unsigned long long key)
{
#pragma unroll
    for (int i = LIST - 1; i > 0; i--) {
        const unsigned long long a = L[i - 1], b = L[i];
        L[i] = key < a ? a : (key < b ? key : b);
    }
    L[0] = key < L[0] ? key : L[0];
}

__device__ __forceinline__ void cluster_sync_all()
{
    asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}
// Bulk copy global -> the same shared offset in every CTA of ctaMask, completing tx on each CTA's barrier.
__device__ __forceinline__ void bulk_load_mc(void* dst, const void* src, unsigned bytes, uint64_t* bar, uint16_t mask)
{
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.multicast::cluster [%0], [%1], %2, [%3], %4;" ::"r"(
            dk::smem_u32(dst)),
        "l"(src), "r"(bytes), "r"(dk::smem_u32(bar)), "h"(mask)
        : "memory");
}
__device__ __forceinline__ void umma_commit_mc(uint64_t* bar, uint16_t mask)
{
    asm volatile(
        "tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.multicast::cluster.b64 [%0], %1;" ::"r"(
            dk::smem_u32(bar)),
        "h"(mask)
        : "memory");
}

// Shared-memory box geometry of the PAIR scheme (must match make_tc_plan): x extent, y extent.
__host__ __device__ constexpr int pair_txb(int m)
{
    return (128 + (m + 1) / 2 * 2 - 1) > (4 * ((m + 3) / 4) + 126) ? (128 + (m + 1) / 2 * 2 - 1)
                                                                     : (4 * ((m + 3) / 4) + 126);
}
// Byte offset of K-step s inside the PAIR pass-1 box ((hi,lo) voxels, 2 per K-step) and pass-2 box
// ((hi(x),hi(x+1)) slots, 4 voxels per K-step); padding steps (zero weights) re-read the last real
// step's voxels (a plane still resident in the z-plane pipeline of dock_tc_skew.cuh).
__host__ __device__ constexpr uint32_t pair_off1(int m, int s, uint32_t row16, uint32_t rowTY)
{
    const int mxp = (m + 1) / 2, t = s < m * m * mxp ? s : m * m * mxp - 1;
    return static_cast<uint32_t>(t / (mxp * m)) * rowTY + static_cast<uint32_t>((t / mxp) % m) * row16 +
           static_cast<uint32_t>(t % mxp) * 32u;
}
__host__ __device__ constexpr uint32_t pair_off2(int m, int s, uint32_t row16, uint32_t rowTY)
{
    const int mxq = (m + 3) / 4, t = s < m * m * mxq ? s : m * m * mxq - 1;
    return static_cast<uint32_t>(t / (mxq * m)) * rowTY + static_cast<uint32_t>((t / mxq) % m) * row16 +
           static_cast<uint32_t>(t % mxq) * 64u;
}

// CL = 1: one CTA per item.  CL = 2: a cluster of two CTAs works on the same rotation block
// (two regions with the same number of tiles); each CTA's producer fetches half of every
// weight chunk and multicasts it into both CTAs' rings, and each MMA warp releases a ring
// slot in both CTAs -- the weight stream from L2 is halved, which lets Q = 2 rows per TMEM
// buffer with NBUF = 2 buffers (epilogue overlapped with the next tile's MMAs).
// PAIR (one channel group): pass 1 reads the (hi, lo) receptor box -> Rhi*Whi + Rlo*Whi over 2 voxels
// per MMA; pass 2 reads a second box whose 16-B slot x holds (Rhi(x), Rhi(x+1)), so one K = 16 MMA
// covers 4 voxels of Rhi*Wlo (chunk LBO = 32 B): 3 MMAs per 4 voxels instead of 4.
template <int M, int Q, int NBUF, int CL, bool PAIR, bool GRID>
__global__ void __launch_bounds__(NTHREADS, 1) k_corr_tc(const __grid_constant__ CUtensorMap tmap,
                                                          const __grid_constant__ CUtensorMap tmap_pair, const TcArgs a)
{
    constexpr int KS = KSTEPS;                 // K-steps per weight-ring stage (one wait/commit per KS steps)
    constexpr unsigned STAGE = KS * WCHUNK;
    static_assert(Q * NBUF * NT <= 512, "TMEM has 512 columns");
    constexpr int MXP = (M + 1) / 2;   // voxel pairs along x (K = 16 = 2 voxels x 8 channels)
    extern __shared__ __align__(1024) unsigned char smem[];
    __shared__ uint64_t bars[2 * 2 + 2 * WSTAGES + NBUF + NBUF * Q];
    __shared__ uint32_t tmem_base_s;
    uint64_t* rec_full = bars;
    uint64_t* rec_empty = bars + 2;
    uint64_t* w_full = bars + 4;
    uint64_t* w_empty = w_full + WSTAGES;
    uint64_t* tm_full = w_empty + WSTAGES;
    uint64_t* tm_empty = tm_full + NBUF;   // [NBUF][Q]: per accumulator row, so the next tile restarts row by row

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int block = blockIdx.x / a.G, region = blockIdx.x % a.G;
    const int tile_begin = region * a.tiles_per_region;
    const int tile_end = min(a.ntiles, tile_begin + a.tiles_per_region);
    const int n_tiles = tile_end - tile_begin;
    unsigned char* rec_smem = smem;
    unsigned char* w_smem = smem + a.n_rec_stages * a.rec_stage_bytes;

    if (threadIdx.x == 0) {
        for (int i = 0; i < 2; i++) {
            dk::mbar_init(&rec_full[i], 1);
            dk::mbar_init(&rec_empty[i], 1);
        }
        for (int i = 0; i < a.wstages; i++) {
            dk::mbar_init(&w_full[i], 1);
            dk::mbar_init(&w_empty[i], CL);
        }
        for (int i = 0; i < NBUF; i++) dk::mbar_init(&tm_full[i], 1);
        for (int i = 0; i < NBUF * Q; i++) dk::mbar_init(&tm_empty[i], a.nepi);
        dk::fence_mbar_init();
    }
    if (warp == 1) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(
            dk::smem_u32(&tmem_base_s)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    if constexpr (CL > 1) cluster_sync_all();   // peers' barriers are initialised before any multicast
    tc_fence_after();
    const uint32_t tmem = tmem_base_s;
    uint32_t crank = 0;
    if constexpr (CL > 1) asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(crank));
    constexpr uint16_t CMASK = (1u << CL) - 1u;

    const bool tr = a.trace != nullptr;
    long long tw0 = 0, tw1 = 0, tw2 = 0, tstart = tr ? clock64() : 0;   // per-role trace accumulators
    if (n_tiles > 0) {
        if (warp == 0) {
            // ------------------------------------------------ TMA producer (warp-converged, one elected lane)
            if (elect_one()) {
                dk::prefetch_tmap(&tmap);
                if constexpr (PAIR) dk::prefetch_tmap(&tmap_pair);
            }
            const unsigned char* wsrc = a.W + static_cast<size_t>(block) * a.nsteps * WCHUNK;
            int ws = 0, wph = 0;                  // weight ring slot / phase
            int wuse = 0;
            auto stream_weights = [&](int s0, int s1) {
                for (int s = s0; s < s1; s += KS) {
                    if (wuse >= a.wstages) twait(&w_empty[ws], wph ^ 1, tr, tw0);
                    if (elect_one()) {
                        dk::mbar_arrive_expect_tx(&w_full[ws], STAGE);
                        if constexpr (CL == 1) {
                            dk::bulk_load(w_smem + static_cast<size_t>(ws) * STAGE,
                                          wsrc + static_cast<size_t>(s) * WCHUNK, STAGE, &w_full[ws]);
                        } else {
                            constexpr unsigned HALF = STAGE / CL;
                            bulk_load_mc(w_smem + static_cast<size_t>(ws) * STAGE + crank * HALF,
                                         wsrc + static_cast<size_t>(s) * WCHUNK + crank * HALF, HALF, &w_full[ws],
                                         CMASK);
                        }
                    }
                    __syncwarp();
                    wuse++;
                    if (++ws == a.wstages) {
                        ws = 0;
                        wph ^= 1;
                    }
                }
            };
            if constexpr (PAIR) {
                // Receptor boxes are issued as soon as their buffer frees: the producer polls the
                // release barriers between weight stages (main(t+1) needs pass 1 of t done, pair(t+1)
                // pass 2 of t), and blocks only right before the first stage that needs a box.
                int pm = 0, pp = 0;   // next main / pair box (tile index) to load
                auto issue_box = [&](int which, int t) {
                    const int tile = tile_begin + t;
                    const int tx = tile % a.ntx, ty = (tile / a.ntx) % a.nty, tz = tile / (a.ntx * a.nty);
                    if (elect_one()) {
                        dk::mbar_arrive_expect_tx(&rec_full[which], a.box_bytes);
                        tma_load_5d(rec_smem + which * a.rec_stage_bytes, which ? &tmap_pair : &tmap, 0, tx * NT,
                                    ty * Q, tz, 0, &rec_full[which]);
                    }
                    __syncwarp();
                };
                auto poll = [&](int ti) {
                    if (pm < n_tiles && pm <= ti + 1 && (pm == 0 || dk::mbar_test(&rec_empty[0], (pm - 1) & 1)))
                        issue_box(0, pm++);
                    if (pp < n_tiles && pp <= ti + 1 && (pp == 0 || dk::mbar_test(&rec_empty[1], (pp - 1) & 1)))
                        issue_box(1, pp++);
                };
                auto ensure = [&](int which, int t) {
                    int& nx = which ? pp : pm;
                    if (nx == t) {
                        if (t > 0) twait(&rec_empty[which], (t - 1) & 1, tr, tw1);
                        issue_box(which, nx++);
                    }
                };
                for (int ti = 0; ti < n_tiles; ti++) {
                    ensure(0, ti);
                    for (int s = 0; s < a.S1p; s += KS) {
                        poll(ti);
                        stream_weights(s, s + KS);
                    }
                    ensure(1, ti);
                    for (int s = a.S1p; s < a.nsteps; s += KS) {
                        poll(ti);
                        stream_weights(s, s + KS);
                    }
                }
            } else {
            for (int ti = 0; ti < n_tiles; ti++) {
                const int tile = tile_begin + ti;
                const int rs = ti % a.n_rec_stages, ruse = ti / a.n_rec_stages;
                if (ruse > 0) twait(&rec_empty[rs], (ruse - 1) & 1, tr, tw1);
                const int tx = tile % a.ntx, ty = (tile / a.ntx) % a.nty, tz = tile / (a.ntx * a.nty);
                unsigned char* rdst = rec_smem + static_cast<size_t>(rs) * a.rec_stage_bytes;
                if (elect_one()) {
                    dk::mbar_arrive_expect_tx(&rec_full[rs], a.G_ch * a.box_bytes);
                    for (int g = 0; g < a.G_ch; g++)
                        tma_load_5d(rdst + static_cast<size_t>(g) * a.box_bytes, &tmap, 0, tx * NT, ty * Q, tz, g,
                                    &rec_full[rs]);
                }
                __syncwarp();
                for (int s = 0; s < a.nsteps; s += KS) {
                    if (wuse >= a.wstages) twait(&w_empty[ws], wph ^ 1, tr, tw0);
                    if (elect_one()) {
                        dk::mbar_arrive_expect_tx(&w_full[ws], STAGE);
                        if constexpr (CL == 1) {
                            dk::bulk_load(w_smem + static_cast<size_t>(ws) * STAGE,
                                          wsrc + static_cast<size_t>(s) * WCHUNK, STAGE, &w_full[ws]);
                        } else {
                            constexpr unsigned HALF = STAGE / CL;
                            bulk_load_mc(w_smem + static_cast<size_t>(ws) * STAGE + crank * HALF,
                                         wsrc + static_cast<size_t>(s) * WCHUNK + crank * HALF, HALF, &w_full[ws],
                                         CMASK);
                        }
                    }
                    __syncwarp();
                    wuse++;
                    if (++ws == a.wstages) {
                        ws = 0;
                        wph ^= 1;
                    }
                }
            }
            }   // !PAIR
            if (tr && elect_one()) {
                atomicAdd(&a.trace[TR_PROD_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                atomicAdd(&a.trace[TR_PROD_WEMPTY], static_cast<unsigned long long>(tw0));
                atomicAdd(&a.trace[TR_PROD_REMPTY], static_cast<unsigned long long>(tw1));
                atomicAdd(&a.trace[TR_CTAS], 1ull);
                atomicAdd(&a.trace[TR_TILES], static_cast<unsigned long long>(n_tiles));
            }
            __syncwarp();
            if constexpr (CL > 1) {
                // drain: every ring slot's last release (from both MMA warps) has arrived before exit
                for (int i = 0; i < min(wuse, a.wstages); i++) {
                    dk::mbar_wait(&w_empty[ws], wph ^ 1);
                    if (++ws == a.wstages) {
                        ws = 0;
                        wph ^= 1;
                    }
                }
            }
        } else if (warp == 1) {
            // ------------------------------------------------ MMA issuer (warp-converged, one elected lane)
            // One elected block per ring stage (KS K-steps x Q rows = KS*Q MMAs): the warp re-converges
            // once per stage, not once per K-step (the re-convergence waits for the tcgen05 issue).
            constexpr uint32_t idesc = umma_idesc(ROT, NT);
            constexpr int MXQ = (M + 3) / 4;   // PAIR pass 2: 4-voxel groups along x
            const uint32_t rec0 = dk::smem_u32(rec_smem), w0 = dk::smem_u32(w_smem);
            const uint64_t dA0 = umma_desc(w0, ROT * 16, 128);                      // + (slot offset >> 4)
            const uint64_t dB0 = umma_desc(rec0, 16, 128);                          // + (voxel offset >> 4)
            const uint64_t dP0 = umma_desc(rec0 + (PAIR ? a.rec_stage_bytes : 0), 32, 128);
            const uint32_t row16 = static_cast<uint32_t>(a.TXB) * 16u;
            const uint32_t rowTY = static_cast<uint32_t>(a.TYB) * row16;
            if constexpr (PAIR && CL == 1) {
            // Lean issue loop: one thread runs the whole schedule (no per-stage warp re-convergence), the
            // stage loops are unrolled so every descriptor offset is an immediate; the tcgen05 queue stays fed.
            constexpr int S1 = M * M * MXP, S1P = (S1 + KS - 1) / KS * KS;
            constexpr int S2 = M * M * MXQ, S2P = (S2 + KS - 1) / KS * KS;
            constexpr uint32_t ROW16 = static_cast<uint32_t>(pair_txb(M)) * 16u;
            constexpr uint32_t ROWTY = static_cast<uint32_t>(Q + M - 1) * ROW16;
            if (elect_one()) {
                uint32_t ws = 0, wph = 0;
                const uint32_t nws = static_cast<uint32_t>(a.wstages);
                for (int ti = 0; ti < n_tiles; ti++) {
                    const int buf = ti % NBUF, buse = ti / NBUF;
                    const uint32_t dcol = tmem + static_cast<uint32_t>(buf * Q * NT);
                    twait(&rec_full[0], ti & 1, tr, tw2);
                    tc_fence_after();
#pragma unroll
                    for (int st = 0; st < S1P / KS; st++) {
                        twait(&w_full[ws], wph, tr, tw1);
                        tc_fence_after();
                        const uint64_t da0 = dA0 + ((ws * STAGE) >> 4);
                        if (st == 0 && buse > 0) {
                            // accumulator rows are released one by one while the epilogue drains them
#pragma unroll
                            for (int q = 0; q < Q; q++) {
                                twait(&tm_empty[buf * Q + q], (buse - 1) & 1, tr, tw0);
                                tc_fence_after();
#pragma unroll
                                for (int ks = 0; ks < KS; ks++)
                                    umma_bf16(dcol + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                              dB0 + ((pair_off1(M, ks, ROW16, ROWTY) + q * ROW16) >> 4), idesc,
                                              ks == 0 ? 0u : 1u);
                            }
                        } else {
#pragma unroll
                            for (int ks = 0; ks < KS; ks++)
#pragma unroll
                                for (int q = 0; q < Q; q++)
                                    umma_bf16(dcol + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                              dB0 + ((pair_off1(M, st * KS + ks, ROW16, ROWTY) + q * ROW16) >> 4),
                                              idesc, (st == 0 && ks == 0) ? 0u : 1u);
                        }
                        umma_commit(&w_empty[ws]);
                        if (++ws == nws) {
                            ws = 0;
                            wph ^= 1;
                        }
                    }
                    umma_commit(&rec_empty[0]);
                    twait(&rec_full[1], ti & 1, tr, tw2);
                    tc_fence_after();
#pragma unroll
                    for (int st = 0; st < S2P / KS; st++) {
                        twait(&w_full[ws], wph, tr, tw1);
                        tc_fence_after();
                        const uint64_t da0 = dA0 + ((ws * STAGE) >> 4);
#pragma unroll
                        for (int ks = 0; ks < KS; ks++)
#pragma unroll
                            for (int q = 0; q < Q; q++)
                                umma_bf16(dcol + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                          dP0 + ((pair_off2(M, st * KS + ks, ROW16, ROWTY) + q * ROW16) >> 4), idesc,
                                          1u);
                        umma_commit(&w_empty[ws]);
                        if (++ws == nws) {
                            ws = 0;
                            wph ^= 1;
                        }
                    }
                    umma_commit(&rec_empty[1]);
                    umma_commit(&tm_full[buf]);
                }
                if (tr) {
                    atomicAdd(&a.trace[TR_MMA_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                    atomicAdd(&a.trace[TR_MMA_TMEMPTY], static_cast<unsigned long long>(tw0));
                    atomicAdd(&a.trace[TR_MMA_WFULL], static_cast<unsigned long long>(tw1));
                    atomicAdd(&a.trace[TR_MMA_RFULL], static_cast<unsigned long long>(tw2));
                }
            }
            __syncwarp();
            } else {
            int ws = 0, wph = 0;
            // B descriptor of K-step s: PAIR pass 1 (kind 0), PAIR pass 2 (kind 1) or the 2-pass scheme (kind 2)
            auto bdesc = [&](int kind, int s, uint32_t rofs) -> uint64_t {
                if (kind == 0) {
                    if (s >= a.S1) return dB0;
                    const int vxp = s % MXP, vy = (s / MXP) % M, vz = s / (MXP * M);
                    return dB0 + ((rofs + vz * rowTY + vy * row16 + vxp * 32u) >> 4);
                }
                if (kind == 1) {
                    if (s >= a.S2) return dP0;
                    const int vxq = s % MXQ, vy = (s / MXQ) % M, vz = s / (MXQ * M);
                    return dP0 + ((vz * rowTY + vy * row16 + vxq * 64u) >> 4);
                }
                const int vxp = s % MXP, vy = (s / MXP) % M, vz = (s / (MXP * M)) % M;
                const int g = s / (MXP * M * M * 2);
                return dB0 + ((rofs + g * a.box_bytes + vz * rowTY + vy * row16 + vxp * 32u) >> 4);
            };
            // rel != nullptr: first stage of a tile whose accumulator rows are still being drained --
            // issue row-major, each row right after the epilogue released it (rel[q], parity relph)
            auto issue_stage = [&](int kind, int s0, uint32_t rofs, uint32_t dcol, bool first, uint64_t* rel,
                                   int relph) {
                twait(&w_full[ws], wph, tr, tw1);
                tc_fence_after();
                const uint64_t da0 = dA0 + ((static_cast<uint32_t>(ws) * STAGE) >> 4);
                if (rel) {
#pragma unroll
                    for (int q = 0; q < Q; q++) {
                        twait(&rel[q], relph, tr, tw0);
                        tc_fence_after();
                        if (elect_one()) {
#pragma unroll
                            for (int ks = 0; ks < KS; ks++)
                                umma_bf16(dcol + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                          bdesc(kind, s0 + ks, rofs) + ((q * row16) >> 4), idesc, ks == 0 ? 0u : 1u);
                        }
                        __syncwarp();
                    }
                } else if (elect_one()) {
#pragma unroll
                    for (int ks = 0; ks < KS; ks++) {
                        const uint64_t db = bdesc(kind, s0 + ks, rofs);
                        const uint64_t da = da0 + ((ks * WCHUNK) >> 4);
#pragma unroll
                        for (int q = 0; q < Q; q++)
                            umma_bf16(dcol + q * NT, da, db + ((q * row16) >> 4), idesc, (first && ks == 0) ? 0u : 1u);
                    }
                }
                __syncwarp();
                if (elect_one()) {
                    if constexpr (CL == 1) umma_commit(&w_empty[ws]);
                    else umma_commit_mc(&w_empty[ws], CMASK);
                }
                __syncwarp();
                if (++ws == a.wstages) {
                    ws = 0;
                    wph ^= 1;
                }
            };
            for (int ti = 0; ti < n_tiles; ti++) {
                const int buf = ti % NBUF, buse = ti / NBUF;
                const uint32_t dcol = tmem + static_cast<uint32_t>(buf * Q * NT);
                if constexpr (PAIR) {
                    twait(&rec_full[0], ti & 1, tr, tw2);
                    tc_fence_after();
                    uint64_t* rel = buse > 0 ? &tm_empty[buf * Q] : nullptr;
                    for (int s = 0; s < a.S1p; s += KS)
                        issue_stage(0, s, 0u, dcol, s == 0, s == 0 ? rel : nullptr, (buse - 1) & 1);
                    if (elect_one()) umma_commit(&rec_empty[0]);
                    __syncwarp();
                    twait(&rec_full[1], ti & 1, tr, tw2);
                    tc_fence_after();
                    for (int s = 0; s < a.S2p; s += KS) issue_stage(1, s, 0u, dcol, false, nullptr, 0);
                    if (elect_one()) {
                        umma_commit(&rec_empty[1]);
                        umma_commit(&tm_full[buf]);
                    }
                    __syncwarp();
                } else {
                    const int rs = ti % a.n_rec_stages, ruse = ti / a.n_rec_stages;
                    twait(&rec_full[rs], ruse & 1, tr, tw2);
                    tc_fence_after();
                    const uint32_t rofs = static_cast<uint32_t>(rs * a.rec_stage_bytes);
                    uint64_t* rel = buse > 0 ? &tm_empty[buf * Q] : nullptr;
                    for (int s = 0; s < a.nsteps; s += KS)
                        issue_stage(2, s, rofs, dcol, s == 0, s == 0 ? rel : nullptr, (buse - 1) & 1);
                    if (elect_one()) {
                        umma_commit(&tm_full[buf]);
                        umma_commit(&rec_empty[rs]);
                    }
                    __syncwarp();
                }
            }
            if (tr && elect_one()) {
                atomicAdd(&a.trace[TR_MMA_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                atomicAdd(&a.trace[TR_MMA_TMEMPTY], static_cast<unsigned long long>(tw0));
                atomicAdd(&a.trace[TR_MMA_WFULL], static_cast<unsigned long long>(tw1));
                atomicAdd(&a.trace[TR_MMA_RFULL], static_cast<unsigned long long>(tw2));
            }
            __syncwarp();
            }   // generic issue loop
        } else {
            // ------------------------------------------------ epilogue warps
            // Warp (quarter, class cls) reads TMEM lanes of its quarter (lane = rotation).  Rows are
            // drained in order q = 0..Q-1 so each accumulator row is released (tm_empty[buf][q]) as soon as
            // its last chunk is in registers, before the chunk is processed; within row q the warp takes the
            // 32-column chunks c = (q + cls + j * nclass) mod 4 ("diagonal" classes: over the Q rows of a
            // tile a class covers one chunk per row, so the cells of a list are spread like a row class).
            const int quarter = warp & 3;
            const int cls = (warp - 2) >> 2;
            const int nclass = a.nepi >> 2;
            constexpr int NCH = NT / 32;                         // 32-column chunks per row
            const int r = quarter * 32 + lane;                  // rotation within the block (TMEM lane)
            const int slot = block * ROT + r;
            const bool rot_ok = slot < a.n_slots;
            unsigned long long lst[LIST];
#pragma unroll
            for (int i = 0; i < LIST; i++) lst[i] = KEY_MAX;
            float th = __int_as_float(0x7f800000);   // score of the list's last key (+inf while not full)
            uint32_t th_t = 0xffffffffu;             // t_lin of the list's last key
            int tx = tile_begin % a.ntx, ty = (tile_begin / a.ntx) % a.nty, tz = tile_begin / (a.ntx * a.nty);
            for (int ti = 0; ti < n_tiles; ti++) {
                const int buf = ti % NBUF, buse = ti / NBUF;
                twait(&tm_full[buf], buse & 1, tr, tw0);
                tc_fence_after();
                if (a.dbg == 1) {   // diagnostic: no TMEM drain
                    __syncwarp();
                    if (lane == 0)
                        for (int q = 0; q < Q; q++) dk::mbar_arrive(&tm_empty[buf * Q + q]);
                } else {
                    const int x0 = tx * NT;
                    for (int q = 0; q < Q; q++) {
                        const int y = ty * Q + q, z = tz;
                        const bool row_ok = rot_ok && y < a.ny && z < a.nz;
                        const uint32_t tbase = static_cast<uint32_t>((z * a.ny + y) * a.nx + x0);
#pragma unroll 1
                        for (int j = 0; j < NCH / nclass; j++) {
                            const int c0 = ((q + cls + j * nclass) & (NCH - 1)) * 32;
                            uint32_t v[32];
                            const long long tl0 = tr ? clock64() : 0;
                            tmem_ld32(tmem + (static_cast<uint32_t>(quarter * 32) << 16) + (buf * Q + q) * NT + c0, v);
                            if (tr) tw1 += clock64() - tl0;
                            if (j == NCH / nclass - 1) {   // the row's last chunk is in registers: release the row
                                tc_fence_before();
                                __syncwarp();
                                if (lane == 0) dk::mbar_arrive(&tm_empty[buf * Q + q]);
                            }
                            if (!row_ok || a.dbg == 2) continue;
                            if constexpr (GRID) {
                                float* out = a.grid + static_cast<size_t>(slot) * a.nx * a.ny * a.nz + tbase;
#pragma unroll
                                for (int jj = 0; jj < 32; jj++)
                                    if (x0 + c0 + jj < a.nx) out[c0 + jj] = __uint_as_float(v[jj]);
                            } else {
                                // fast check: one FMNMX per value; the insertion path is rare after warm-up
                                float mn = __uint_as_float(v[0]);
#pragma unroll
                                for (int jj = 1; jj < 32; jj++) mn = fminf(mn, __uint_as_float(v[jj]));
                                // exact gate: a strictly better score, or a tie that could carry a smaller t_lin
                                if (mn < th || (mn == th && tbase + c0 < th_t)) {
                                    // rare path: bitmask of candidates, each extracted with a 5-level select tree
                                    const int jmax = min(32, a.nx - x0 - c0);
                                    uint32_t msk = 0;
#pragma unroll
                                    for (int jj = 0; jj < 32; jj++)
                                        msk |= (__uint_as_float(v[jj]) <= th && jj < jmax) ? (1u << jj) : 0u;
                                    while (msk) {
                                        const int jj = __ffs(msk) - 1;
                                        msk &= msk - 1;
                                        const float sv = __uint_as_float(select32(v, jj));
                                        if (sv <= th) {
                                            const unsigned long long key = dk::make_key(sv, tbase + c0 + jj);
                                            if (key < lst[LIST - 1]) {
                                                list_insert(lst, key);
                                                th = dk::key_score_bound(static_cast<uint32_t>(lst[LIST - 1] >> 32));
                                                th_t = static_cast<uint32_t>(lst[LIST - 1] & 0xffffffffu);
                                            }
                                        }
                                    }
                                }
                            }
                        }
                    }
                }
                if (++tx == a.ntx) {
                    tx = 0;
                    if (++ty == a.nty) {
                        ty = 0;
                        tz++;
                    }
                }
            }
            if (tr && lane == 0) {
                atomicAdd(&a.trace[TR_EPI_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                atomicAdd(&a.trace[TR_EPI_TMFULL], static_cast<unsigned long long>(tw0));
                atomicAdd(&a.trace[TR_EPI_LDTM], static_cast<unsigned long long>(tw1));
                atomicAdd(&a.trace[TR_EPI_WARPS], 1ull);
            }
            if constexpr (!GRID) {
                if (rot_ok) {
                    // bound: k list entries pairwise farther than 2*rho apart.
                    // Loops over the register list are fully unrolled (static indices keep it in registers).
                    unsigned long long Tw = KEY_MAX;
                    uint32_t chosen[32];
                    int nc = 0;
#pragma unroll
                    for (int i = 0; i < LIST; i++) {
                        const unsigned long long key = lst[i];
                        if (key != KEY_MAX && nc < a.k) {
                            const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
                            bool far = true;
                            for (int c = 0; c < nc; c++)
                                far = far && dk::cheb_cyc(t, chosen[c], a.nx, a.ny, a.nz) > 2 * a.rho;
                            if (far) {
                                chosen[nc] = t;
                                nc++;
                                if (nc == a.k) Tw = key;
                            }
                        }
                    }
                    const unsigned long long old = atomicMin(&a.T[slot], Tw);
                    const unsigned long long Tn = old < Tw ? old : Tw;
                    atomicMin(&a.mu[slot], lst[LIST - 1]);
#pragma unroll
                    for (int i = 0; i < LIST; i++) {
                        const unsigned long long key = lst[i];
                        if (key != KEY_MAX && key <= Tn) {
                            const unsigned pos = atomicAdd(&a.cnt[slot], 1u);
                            if (pos < static_cast<unsigned>(a.cap)) a.cand[static_cast<size_t>(slot) * a.cap + pos] = key;
                        }
                    }
                }
            }
        }
    }
    tc_fence_before();
    __syncthreads();
    if (warp == 1) asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
    if constexpr (CL > 1) cluster_sync_all();
}

// ------------------------------------------------------------------ data preparation

// bf16 split of the padded receptor: Rb[g][Z][Y][X][8] = (hi_0..3, lo_0..3) of channels 4g..4g+3
__global__ void k_pack_receptor_tc(const float* __restrict__ R, uint16_t* __restrict__ Rb, int nx, int ny, int nz,
                                   int Xp, int Yp, int Zp, int P, int G_ch)
{
    const size_t total = static_cast<size_t>(G_ch) * Zp * Yp * Xp;
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<size_t>(gridDim.x) * blockDim.x) {
        const int X = static_cast<int>(i % Xp);
        size_t rr = i / Xp;
        const int Y = static_cast<int>(rr % Yp);
        rr /= Yp;
        const int Z = static_cast<int>(rr % Zp);
        const int g = static_cast<int>(rr / Zp);
        uint16_t out[8];
#pragma unroll
        for (int c = 0; c < 4; c++) {
            const int p = 4 * g + c;
            float f = 0.f;
            if (p < P) f = R[((static_cast<size_t>(p) * nz + Z % nz) * ny + Y % ny) * nx + X % nx];
            const __nv_bfloat16 hi = __float2bfloat16_rn(f);
            const __nv_bfloat16 lo = __float2bfloat16_rn(f - __bfloat162float(hi));
            out[c] = __bfloat16_as_ushort(hi);
            out[4 + c] = __bfloat16_as_ushort(lo);
        }
        uint4 pk;
        pk.x = out[0] | (static_cast<uint32_t>(out[1]) << 16);
        pk.y = out[2] | (static_cast<uint32_t>(out[3]) << 16);
        pk.z = out[4] | (static_cast<uint32_t>(out[5]) << 16);
        pk.w = out[6] | (static_cast<uint32_t>(out[7]) << 16);
        reinterpret_cast<uint4*>(Rb)[i] = pk;
    }
}

// Folded weights Lw [batch][P][m^3][RB] (k_voxelize output) -> A operand [block][step][chunk][rot][8].
__global__ void k_pack_weights_tc(const float* __restrict__ Lw, unsigned char* __restrict__ W, int n_slots, int P,
                                  int G_ch, int m, int nsteps)
{
    const int MXP = (m + 1) / 2, m3 = m * m * m;
    const long long n_blocks = (n_slots + ROT - 1) / ROT;
    const long long total = n_blocks * nsteps * 2 * ROT;   // one thread per (block, step, chunk, rot) 16-B row
    for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<long long>(gridDim.x) * blockDim.x) {
        const int r = static_cast<int>(i % ROT);
        const int c = static_cast<int>((i / ROT) % 2);
        const int s = static_cast<int>((i / (2 * ROT)) % nsteps);
        const long long blk = i / (2LL * ROT * nsteps);
        const int vxp = s % MXP, vy = (s / MXP) % m, vz = (s / (MXP * m)) % m;
        const int pass = (s / (MXP * m * m)) % 2, g = s / (MXP * m * m * 2);
        const int vx = 2 * vxp + c;
        const long long slot = blk * ROT + r;
        uint16_t out[8] = {0, 0, 0, 0, 0, 0, 0, 0};
        if (slot < n_slots && vx < m) {
            const int v = (vz * m + vy) * m + vx;
#pragma unroll
            for (int cc = 0; cc < 4; cc++) {
                const int p = 4 * g + cc;
                if (p >= P) continue;
                const float f = Lw[((static_cast<size_t>(slot / dk::RB) * P + p) * m3 + v) * dk::RB + slot % dk::RB];
                const __nv_bfloat16 hi = __float2bfloat16_rn(f);
                const __nv_bfloat16 lo = __float2bfloat16_rn(f - __bfloat162float(hi));
                if (pass == 0) {
                    out[cc] = __bfloat16_as_ushort(hi);
                    out[4 + cc] = __bfloat16_as_ushort(hi);
                } else {
                    out[cc] = __bfloat16_as_ushort(lo);
                }
            }
        }
        uint4 pk;
        pk.x = out[0] | (static_cast<uint32_t>(out[1]) << 16);
        pk.y = out[2] | (static_cast<uint32_t>(out[3]) << 16);
        pk.z = out[4] | (static_cast<uint32_t>(out[5]) << 16);
        pk.w = out[6] | (static_cast<uint32_t>(out[7]) << 16);
        reinterpret_cast<uint4*>(W)[i] = pk;
    }
}

// PAIR scheme, second receptor copy: slot X holds (Rhi_0..3(X), Rhi_0..3(X+1)) of channels 0..3.
__global__ void k_pack_receptor_pair_tc(const float* __restrict__ R, uint16_t* __restrict__ Rb, int nx, int ny, int nz,
                                        int Xp, int Yp, int Zp, int P)
{
    const size_t total = static_cast<size_t>(Zp) * Yp * Xp;
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<size_t>(gridDim.x) * blockDim.x) {
        const int X = static_cast<int>(i % Xp);
        size_t rr = i / Xp;
        const int Y = static_cast<int>(rr % Yp);
        const int Z = static_cast<int>(rr / Yp);
        uint16_t out[8];
#pragma unroll
        for (int c = 0; c < 8; c++) {
            const int p = c & 3, dx = c >> 2;
            float f = 0.f;
            if (p < P) f = R[((static_cast<size_t>(p) * nz + Z % nz) * ny + Y % ny) * nx + (X + dx) % nx];
            out[c] = __bfloat16_as_ushort(__float2bfloat16_rn(f));
        }
        uint4 pk;
        pk.x = out[0] | (static_cast<uint32_t>(out[1]) << 16);
        pk.y = out[2] | (static_cast<uint32_t>(out[3]) << 16);
        pk.z = out[4] | (static_cast<uint32_t>(out[5]) << 16);
        pk.w = out[6] | (static_cast<uint32_t>(out[7]) << 16);
        reinterpret_cast<uint4*>(Rb)[i] = pk;
    }
}

// PAIR scheme A operand: steps [0, S1p) = pass 1 chunks (Whi(vx), Whi(vx)), vx = 2 vxp + c;
// steps [S1p, S1p + S2p) = pass 2 chunks (Wlo(vx0), Wlo(vx0 + 1)), vx0 = 4 vxq + 2c; padding = 0.
__global__ void k_pack_weights_tc_pair(const float* __restrict__ Lw, unsigned char* __restrict__ W, int n_slots, int P,
                                       int m, int S1, int S1p, int S2, int S2p)
{
    const int MXP = (m + 1) / 2, MXQ = (m + 3) / 4, m3 = m * m * m, nsteps = S1p + S2p;
    const long long n_blocks = (n_slots + ROT - 1) / ROT;
    const long long total = n_blocks * nsteps * 2 * ROT;
    for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<long long>(gridDim.x) * blockDim.x) {
        const int r = static_cast<int>(i % ROT);
        const int c = static_cast<int>((i / ROT) % 2);
        const int s = static_cast<int>((i / (2 * ROT)) % nsteps);
        const long long blk = i / (2LL * ROT * nsteps);
        const long long slot = blk * ROT + r;
        uint16_t out[8] = {0, 0, 0, 0, 0, 0, 0, 0};
        auto wval = [&](int vz, int vy, int vx, int p) -> float {
            if (vx >= m || p >= P) return 0.f;
            const int v = (vz * m + vy) * m + vx;
            return Lw[((static_cast<size_t>(slot / dk::RB) * P + p) * m3 + v) * dk::RB + slot % dk::RB];
        };
        if (slot < n_slots) {
            if (s < S1) {
                const int vxp = s % MXP, vy = (s / MXP) % m, vz = s / (MXP * m);
                const int vx = 2 * vxp + c;
#pragma unroll
                for (int p = 0; p < 4; p++) {
                    const __nv_bfloat16 hi = __float2bfloat16_rn(wval(vz, vy, vx, p));
                    out[p] = out[4 + p] = __bfloat16_as_ushort(hi);
                }
            } else if (s >= S1p && s - S1p < S2) {
                const int t = s - S1p;
                const int vxq = t % MXQ, vy = (t / MXQ) % m, vz = t / (MXQ * m);
                const int vx0 = 4 * vxq + 2 * c;
#pragma unroll
                for (int p = 0; p < 4; p++) {
#pragma unroll
                    for (int d = 0; d < 2; d++) {
                        const float f = wval(vz, vy, vx0 + d, p);
                        const __nv_bfloat16 hi = __float2bfloat16_rn(f);
                        const __nv_bfloat16 lo = __float2bfloat16_rn(f - __bfloat162float(hi));
                        out[4 * d + p] = __bfloat16_as_ushort(lo);
                    }
                }
            }
        }
        uint4 pk;
        pk.x = out[0] | (static_cast<uint32_t>(out[1]) << 16);
        pk.y = out[2] | (static_cast<uint32_t>(out[3]) << 16);
        pk.z = out[4] | (static_cast<uint32_t>(out[5]) << 16);
        pk.w = out[6] | (static_cast<uint32_t>(out[7]) << 16);
        reinterpret_cast<uint4*>(W)[i] = pk;
    }
}

// ------------------------------------------------------------------ variant 3: cta_group::2

__device__ __forceinline__ void umma_bf16_2sm(uint32_t d_tmem, uint64_t a, uint64_t b, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\tsetp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::2.kind::f16 [%0], %1, %2, %3, p;\n\t}\n" ::"r"(d_tmem),
        "l"(a), "l"(b), "r"(idesc), "r"(acc)
        : "memory");
}
__device__ __forceinline__ void umma_commit_2sm_mc(uint64_t* bar, uint16_t mask)
{
    asm volatile(
        "tcgen05.commit.cta_group::2.mbarrier::arrive::one.shared::cluster.multicast::cluster.b64 [%0], %1;" ::"r"(
            dk::smem_u32(bar)),
        "h"(mask)
        : "memory");
}
// Arrive on the barrier at the same shared-memory offset in CTA `rank` of the cluster.
__device__ __forceinline__ void mbar_arrive_remote(uint64_t* bar, uint32_t rank)
{
    asm volatile(
        "{\n\t.reg .b32 ra;\n\tmapa.shared::cluster.u32 ra, %0, %1;\n\t"
        "mbarrier.arrive.release.cluster.shared::cluster.b64 _, [ra];\n\t}\n" ::"r"(dk::smem_u32(bar)),
        "r"(rank)
        : "memory");
}

// Variant 3: a CTA pair runs 256 rotations (its two blocks) against 4 receptor rows per tile,
// each CTA holding 2 of the rows.  The leader issues tcgen05.mma.cta_group::2 M = 256 x N = 256:
// A = each CTA's own 128 rotations, B = CTA0's row q (N 0..127) and CTA1's row q (N 128..255),
// D = each CTA's TMEM [128 rotations][2 accumulators x 256 columns].  Per SM this halves the
// shared-memory operand reads and the MMA instructions of variant 1.  Loads complete on local
// barriers; the peer's MMA warp relays "stage full" to the leader with a remote arrive, and the
// leader's commits release stages in both CTAs (multicast).
template <int M, bool GRID>
__global__ void __launch_bounds__(NTHREADS, 1) k_corr_tc2(const __grid_constant__ CUtensorMap tmap,
                                                           const __grid_constant__ CUtensorMap tmap_pair, const TcArgs a)
{
    constexpr int KS = KSTEPS;
    constexpr unsigned STAGE = KS * WCHUNK;
    constexpr int QL = 2;                 // receptor rows per CTA per tile; the pair covers 4
    constexpr int MXP = (M + 1) / 2, MXQ = (M + 3) / 4;
    extern __shared__ __align__(1024) unsigned char smem[];
    __shared__ uint64_t bars[2 * 2 + 2 * WSTAGES + 2 + 2 + WSTAGES];
    __shared__ uint32_t tmem_base_s;
    uint64_t* rec_full = bars;
    uint64_t* rec_empty = bars + 2;
    uint64_t* w_full = bars + 4;
    uint64_t* w_empty = w_full + WSTAGES;
    uint64_t* tm_full = w_empty + WSTAGES;
    uint64_t* tm_empty = tm_full + 1;
    uint64_t* peer_rec = tm_empty + 1;    // leader only: peer's receptor buffers landed
    uint64_t* peer_w = peer_rec + 2;      // leader only: peer's weight stages landed

    uint32_t crank;
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(crank));
    const bool leader = crank == 0;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int pitem = blockIdx.x >> 1;
    const int bp = pitem / a.G, region = pitem % a.G;
    const int block = 2 * bp + static_cast<int>(crank);
    const int tile_begin = region * a.tiles_per_region;
    const int tile_end = min(a.ntiles, tile_begin + a.tiles_per_region);
    const int n_tiles = tile_end - tile_begin;
    unsigned char* rec_smem = smem;
    unsigned char* w_smem = smem + 2 * a.rec_stage_bytes;

    if (threadIdx.x == 0) {
        for (int i = 0; i < 2; i++) {
            dk::mbar_init(&rec_full[i], 1);
            dk::mbar_init(&rec_empty[i], 1);
            dk::mbar_init(&peer_rec[i], 1);
        }
        for (int i = 0; i < a.wstages; i++) {
            dk::mbar_init(&w_full[i], 1);
            dk::mbar_init(&w_empty[i], 1);
            dk::mbar_init(&peer_w[i], 1);
        }
        dk::mbar_init(&tm_full[0], 1);
        dk::mbar_init(&tm_empty[0], 2 * a.nepi);
        dk::fence_mbar_init();
    }
    if (warp == 1) {
        asm volatile("tcgen05.alloc.cta_group::2.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(
            dk::smem_u32(&tmem_base_s)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::2.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    cluster_sync_all();
    tc_fence_after();
    const uint32_t tmem = tmem_base_s;
    const bool tr = a.trace != nullptr;
    long long tw0 = 0, tw1 = 0, tw2 = 0, tstart = tr ? clock64() : 0;

    if (n_tiles > 0) {
        if (warp == 0) {
            // ------------------------------------------------ TMA producer (both CTAs, local data)
            if (elect_one()) {
                dk::prefetch_tmap(&tmap);
                dk::prefetch_tmap(&tmap_pair);
            }
            const unsigned char* wsrc = a.W + static_cast<size_t>(block) * a.nsteps * WCHUNK;
            int ws = 0, wph = 0, wuse = 0;
            auto stream_weights = [&](int s0, int s1) {
                for (int s = s0; s < s1; s += KS) {
                    if (wuse >= a.wstages) twait(&w_empty[ws], wph ^ 1, tr, tw0);
                    if (elect_one()) {
                        dk::mbar_arrive_expect_tx(&w_full[ws], STAGE);
                        dk::bulk_load(w_smem + static_cast<size_t>(ws) * STAGE, wsrc + static_cast<size_t>(s) * WCHUNK,
                                      STAGE, &w_full[ws]);
                    }
                    __syncwarp();
                    wuse++;
                    if (++ws == a.wstages) {
                        ws = 0;
                        wph ^= 1;
                    }
                }
            };
            int pm = 0, pp = 0;
            auto issue_box = [&](int which, int t) {
                const int tile = tile_begin + t;
                const int tx = tile % a.ntx, ty = (tile / a.ntx) % a.nty, tz = tile / (a.ntx * a.nty);
                const int y0 = ty * (2 * QL) + QL * static_cast<int>(crank);
                if (elect_one()) {
                    dk::mbar_arrive_expect_tx(&rec_full[which], a.box_bytes);
                    tma_load_5d(rec_smem + which * a.rec_stage_bytes, which ? &tmap_pair : &tmap, 0, tx * NT, y0, tz,
                                0, &rec_full[which]);
                }
                __syncwarp();
            };
            auto poll = [&](int ti) {
                if (pm < n_tiles && pm <= ti + 1 && (pm == 0 || dk::mbar_test(&rec_empty[0], (pm - 1) & 1)))
                    issue_box(0, pm++);
                if (pp < n_tiles && pp <= ti + 1 && (pp == 0 || dk::mbar_test(&rec_empty[1], (pp - 1) & 1)))
                    issue_box(1, pp++);
            };
            auto ensure = [&](int which, int t) {
                int& nx = which ? pp : pm;
                if (nx == t) {
                    if (t > 0) twait(&rec_empty[which], (t - 1) & 1, tr, tw1);
                    issue_box(which, nx++);
                }
            };
            for (int ti = 0; ti < n_tiles; ti++) {
                ensure(0, ti);
                for (int s = 0; s < a.S1p; s += KS) {
                    poll(ti);
                    stream_weights(s, s + KS);
                }
                ensure(1, ti);
                for (int s = a.S1p; s < a.nsteps; s += KS) {
                    poll(ti);
                    stream_weights(s, s + KS);
                }
            }
            if (tr && leader && elect_one()) {
                atomicAdd(&a.trace[TR_PROD_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                atomicAdd(&a.trace[TR_PROD_WEMPTY], static_cast<unsigned long long>(tw0));
                atomicAdd(&a.trace[TR_PROD_REMPTY], static_cast<unsigned long long>(tw1));
                atomicAdd(&a.trace[TR_CTAS], 1ull);
                atomicAdd(&a.trace[TR_TILES], static_cast<unsigned long long>(n_tiles));
            }
            __syncwarp();
        } else if (warp == 1) {
            if (!leader) {
                // ------------------------------------------------ relay: tell the leader our stages landed
                int ws = 0, wph = 0;
                auto relay_stages = [&](int n) {
                    for (int s = 0; s < n; s += KS) {
                        dk::mbar_wait(&w_full[ws], wph);
                        if (elect_one()) mbar_arrive_remote(&peer_w[ws], 0);
                        __syncwarp();
                        if (++ws == a.wstages) {
                            ws = 0;
                            wph ^= 1;
                        }
                    }
                };
                for (int ti = 0; ti < n_tiles; ti++) {
                    dk::mbar_wait(&rec_full[0], ti & 1);
                    if (elect_one()) mbar_arrive_remote(&peer_rec[0], 0);
                    __syncwarp();
                    relay_stages(a.S1p);
                    dk::mbar_wait(&rec_full[1], ti & 1);
                    if (elect_one()) mbar_arrive_remote(&peer_rec[1], 0);
                    __syncwarp();
                    relay_stages(a.S2p);
                }
            } else {
                // ------------------------------------------------ leader: MMA issue for the pair
                constexpr uint32_t idesc = umma_idesc(2 * ROT, 2 * NT);
                constexpr uint16_t PAIRMASK = 3;
                const uint32_t rec0 = dk::smem_u32(rec_smem), w0 = dk::smem_u32(w_smem);
                const uint64_t dA0 = umma_desc(w0, ROT * 16, 128);
                const uint64_t dB0 = umma_desc(rec0, 16, 128);
                const uint64_t dP0 = umma_desc(rec0 + a.rec_stage_bytes, 32, 128);
                const uint32_t row16 = static_cast<uint32_t>(a.TXB) * 16u;
                const uint32_t rowTY = static_cast<uint32_t>(a.TYB) * row16;
                int ws = 0, wph = 0;
                auto issue_stage = [&](int kind, int s0, bool first) {
                    twait(&w_full[ws], wph, tr, tw1);
                    twait(&peer_w[ws], wph, tr, tw1);
                    tc_fence_after();
                    if (elect_one()) {
                        const uint64_t da0 = dA0 + ((static_cast<uint32_t>(ws) * STAGE) >> 4);
#pragma unroll
                        for (int ks = 0; ks < KS; ks++) {
                            const int s = s0 + ks;
                            uint64_t db;
                            if (kind == 0) {
                                const int vxp = s % MXP, vy = (s / MXP) % M, vz = s / (MXP * M);
                                db = s < a.S1 ? dB0 + ((vz * rowTY + vy * row16 + vxp * 32u) >> 4) : dB0;
                            } else {
                                const int vxq = s % MXQ, vy = (s / MXQ) % M, vz = s / (MXQ * M);
                                db = s < a.S2 ? dP0 + ((vz * rowTY + vy * row16 + vxq * 64u) >> 4) : dP0;
                            }
                            const uint64_t da = da0 + ((ks * WCHUNK) >> 4);
#pragma unroll
                            for (int q = 0; q < QL; q++)
                                umma_bf16_2sm(tmem + q * 2 * NT, da, db + ((q * row16) >> 4), idesc,
                                              (first && ks == 0) ? 0u : 1u);
                        }
                        umma_commit_2sm_mc(&w_empty[ws], PAIRMASK);
                    }
                    __syncwarp();
                    if (++ws == a.wstages) {
                        ws = 0;
                        wph ^= 1;
                    }
                };
                for (int ti = 0; ti < n_tiles; ti++) {
                    twait(&rec_full[0], ti & 1, tr, tw2);
                    twait(&peer_rec[0], ti & 1, tr, tw2);
                    if (ti > 0) twait(&tm_empty[0], (ti - 1) & 1, tr, tw0);
                    tc_fence_after();
                    for (int s = 0; s < a.S1p; s += KS) issue_stage(0, s, s == 0);
                    if (elect_one()) umma_commit_2sm_mc(&rec_empty[0], PAIRMASK);
                    __syncwarp();
                    twait(&rec_full[1], ti & 1, tr, tw2);
                    twait(&peer_rec[1], ti & 1, tr, tw2);
                    tc_fence_after();
                    for (int s = 0; s < a.S2p; s += KS) issue_stage(1, s, false);
                    if (elect_one()) {
                        umma_commit_2sm_mc(&rec_empty[1], PAIRMASK);
                        umma_commit_2sm_mc(&tm_full[0], PAIRMASK);
                    }
                    __syncwarp();
                }
                if (tr && elect_one()) {
                    atomicAdd(&a.trace[TR_MMA_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                    atomicAdd(&a.trace[TR_MMA_TMEMPTY], static_cast<unsigned long long>(tw0));
                    atomicAdd(&a.trace[TR_MMA_WFULL], static_cast<unsigned long long>(tw1));
                    atomicAdd(&a.trace[TR_MMA_RFULL], static_cast<unsigned long long>(tw2));
                }
                __syncwarp();
            }
        } else if (warp < 2 + a.nepi) {
            // ------------------------------------------------ epilogue warps (both CTAs)
            const int quarter = warp & 3;
            const int cls = (warp - 2) >> 2;                 // 0..3 -> (accumulator q, CTA half)
            const int nclass = a.nepi >> 2;
            const int r = quarter * 32 + lane;
            const int slot = block * ROT + r;
            const bool rot_ok = slot < a.n_slots;
            unsigned long long lst[LIST];
#pragma unroll
            for (int i = 0; i < LIST; i++) lst[i] = KEY_MAX;
            float th = __int_as_float(0x7f800000);
            uint32_t th_t = 0xffffffffu;
            for (int ti = 0; ti < n_tiles; ti++) {
                const int tile = tile_begin + ti;
                twait(&tm_full[0], ti & 1, tr, tw0);
                tc_fence_after();
                if (a.dbg == 1) {   // diagnostic: no TMEM drain
                    __syncwarp();
                    if (lane == 0) {
                        if (leader) dk::mbar_arrive(&tm_empty[0]);
                        else mbar_arrive_remote(&tm_empty[0], 0);
                    }
                    continue;
                }
                const int tx = tile % a.ntx, ty = (tile / a.ntx) % a.nty, tz = tile / (a.ntx * a.nty);
                for (int c4 = cls; c4 < 4; c4 += nclass) {
                    const int q = c4 >> 1, half = c4 & 1;
                    const int y = ty * (2 * QL) + QL * half + q, z = tz;
                    const bool row_ok = rot_ok && y < a.ny && z < a.nz;
                    const int x0 = tx * NT;
                    const uint32_t tbase = static_cast<uint32_t>((z * a.ny + y) * a.nx + x0);
#pragma unroll 1
                    for (int c0 = 0; c0 < NT; c0 += 32) {
                        uint32_t v[32];
                        const long long tl0 = tr ? clock64() : 0;
                        tmem_ld32(tmem + (static_cast<uint32_t>(quarter * 32) << 16) + q * 2 * NT + half * NT + c0, v);
                        if (tr) tw1 += clock64() - tl0;
                        if (!row_ok || a.dbg == 2) continue;
                        if constexpr (GRID) {
                            float* out = a.grid + static_cast<size_t>(slot) * a.nx * a.ny * a.nz + tbase;
#pragma unroll
                            for (int j = 0; j < 32; j++)
                                if (x0 + c0 + j < a.nx) out[c0 + j] = __uint_as_float(v[j]);
                        } else {
                            float mn = __uint_as_float(v[0]);
#pragma unroll
                            for (int j = 1; j < 32; j++) mn = fminf(mn, __uint_as_float(v[j]));
                            if (mn < th || (mn == th && tbase + c0 < th_t)) {
                                const int jmax = min(32, a.nx - x0 - c0);
                                uint32_t msk = 0;
#pragma unroll
                                for (int j = 0; j < 32; j++)
                                    msk |= (__uint_as_float(v[j]) <= th && j < jmax) ? (1u << j) : 0u;
                                while (msk) {
                                    const int j = __ffs(msk) - 1;
                                    msk &= msk - 1;
                                    const float sv = __uint_as_float(select32(v, j));
                                    if (sv <= th) {
                                        const unsigned long long key = dk::make_key(sv, tbase + c0 + j);
                                        if (key < lst[LIST - 1]) {
                                            list_insert(lst, key);
                                            th = dk::key_score_bound(static_cast<uint32_t>(lst[LIST - 1] >> 32));
                                            th_t = static_cast<uint32_t>(lst[LIST - 1] & 0xffffffffu);
                                        }
                                    }
                                }
                            }
                        }
                    }
                }
                tc_fence_before();
                __syncwarp();
                if (lane == 0) {
                    if (leader) dk::mbar_arrive(&tm_empty[0]);
                    else mbar_arrive_remote(&tm_empty[0], 0);
                }
            }
            if (tr && leader && lane == 0) {
                atomicAdd(&a.trace[TR_EPI_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                atomicAdd(&a.trace[TR_EPI_TMFULL], static_cast<unsigned long long>(tw0));
                atomicAdd(&a.trace[TR_EPI_LDTM], static_cast<unsigned long long>(tw1));
                atomicAdd(&a.trace[TR_EPI_WARPS], 1ull);
            }
            if constexpr (!GRID) {
                if (rot_ok) {
                    unsigned long long Tw = KEY_MAX;
                    uint32_t chosen[32];
                    int nc = 0;
#pragma unroll
                    for (int i = 0; i < LIST; i++) {
                        const unsigned long long key = lst[i];
                        if (key != KEY_MAX && nc < a.k) {
                            const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
                            bool far = true;
                            for (int c = 0; c < nc; c++)
                                far = far && dk::cheb_cyc(t, chosen[c], a.nx, a.ny, a.nz) > 2 * a.rho;
                            if (far) {
                                chosen[nc] = t;
                                nc++;
                                if (nc == a.k) Tw = key;
                            }
                        }
                    }
                    const unsigned long long old = atomicMin(&a.T[slot], Tw);
                    const unsigned long long Tn = old < Tw ? old : Tw;
                    atomicMin(&a.mu[slot], lst[LIST - 1]);
#pragma unroll
                    for (int i = 0; i < LIST; i++) {
                        const unsigned long long key = lst[i];
                        if (key != KEY_MAX && key <= Tn) {
                            const unsigned pos = atomicAdd(&a.cnt[slot], 1u);
                            if (pos < static_cast<unsigned>(a.cap)) a.cand[static_cast<size_t>(slot) * a.cap + pos] = key;
                        }
                    }
                }
            }
        }
    }
    tc_fence_before();
    __syncthreads();
    cluster_sync_all();
    if (warp == 1) asm volatile("tcgen05.dealloc.cta_group::2.sync.aligned.b32 %0, 512;" ::"r"(tmem));
    cluster_sync_all();
}

}  // namespace tc

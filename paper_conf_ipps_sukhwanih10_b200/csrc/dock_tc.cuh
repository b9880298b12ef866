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
// A (weights, K-major) streams through a <= 16-stage mbarrier ring (4 KB per K-step) and is
// reused by the Q translation rows of a tile; D lives in TMEM (Q x NTT columns).
// Two kernels: variant 1 (k_corr_tc: one channel group, both receptor boxes resident, NTT = 128) and
// variant 2 (k_corr_tcs: any number of channel groups and m <= 8, receptor streamed z-plane by
// z-plane through a ring, NTT in {64, 128, 160}).
// Epilogue: one thread per (rotation, half of the rows) reads its TMEM lane with
// tcgen05.ld and keeps an exact per-thread top-LIST key list (no score grid in HBM),
// published at item end exactly like the FFMA engine (k_merge is shared).
#pragma once
#include <cuda_bf16.h>

#include <type_traits>
#include <utility>

#include "dock_kernels.cuh"

namespace tc {

using dk::KEY_MAX;

constexpr int ROT = 128;        // rotations per block (MMA M)
constexpr int NT = 128;         // translations per row (MMA N)
#ifndef DOCK_TC_NEPI_MAX
#define DOCK_TC_NEPI_MAX 8
#endif
#ifndef DOCK_TC_STAIR
#define DOCK_TC_STAIR 3
#endif
constexpr int NEPI_MAX = DOCK_TC_NEPI_MAX;   // epilogue warps: a.nepi in {4, 8} (1 or 2 per TMEM lane quarter; 8 measured best: 168 registers per thread, 2 row classes)
constexpr int NTHREADS = (3 + NEPI_MAX) * 32;   // launch bound; both variants launch (3 + a.nepi) * 32 threads
constexpr int WSTAGES = 16;     // max weight ring depth (runtime a.wstages <= 16; 16 x 4 KB covers the L2 latency)
constexpr int WCHUNK = 2 * ROT * 16;   // bytes of one K-step of A (2 K-chunks x 128 rotations x 16 B)
#ifndef DOCK_TC_KSTEPS
#define DOCK_TC_KSTEPS 4
#endif
constexpr int KSTEPS = DOCK_TC_KSTEPS;   // K-steps of A per ring stage (KSTEPS * Q MMAs per stage)
constexpr int LIST = 16;        // per-thread candidate list (exact top-LIST keys of one rotation and row class)

struct TcArgs {
    int nx, ny, nz;
    int ntx, nty, ntz, ntiles;  // tiles: NTT x Q rows (y) x 1 (z)
    int G_ch;                   // channel groups of 4
    int n_slots, G, tiles_per_region;
    int chunk;                  // variant 1: > 0 -> dynamic scheduling: persistent CTAs (one per SM) take
                                // chunks of `chunk` tiles of one rotation block (see k_corr_tc);
                                // 0 -> CTA = (block, region) with G regions of tiles_per_region tiles
    unsigned long long* sched;  // [1 + gridDim.x]: CTAs done, chunks taken per segment (zero between
                                // launches: the last CTA to finish resets them)
    int nsteps;                 // K-steps of A per tile (all passes / units, padded to whole ring stages)
    const unsigned char* W;     // [block][step][WCHUNK]
    // variant 1 occupancy schedule (k_tc_block_tables): per rotation block only the K-steps where some
    // rotation of the block has a nonzero probe weight (plus zero-weight padding to whole ring stages)
    const int4* kinfo;          // [block]: (ring stages of the compacted A stream, -, active K-step mask lo, hi)
    const int* perm;            // [block * ROT]: block position -> unit slot (occupancy clustering); nullptr =
                                // identity
    const int* blkmap;          // block sharding: [local block] -> block of the call's block order; nullptr = identity
    int n_blocks;               // blocks this launch processes (local count under block sharding; 0 = all)
    const long long* seg;       // [gridDim.x + 1]: dynamic scheduler segment boundaries (chunk ids) balanced by the
                                // blocks' schedule lengths (k_tc_segments); nullptr = equal chunk counts
    int box_bytes;              // bytes of one receptor TMA box (variant 1: the main box; variant 2: one z-plane)
    int box_bytes_pair;         // variant 1: bytes of the pair box
    int box_bytes_b, rec_off_b; // variant 1: the main box is two half-boxes, z planes [0, mh) at 0 (box_bytes) and
                                // [mh, m) at rec_off_b (box_bytes_b, 0 when m = 1), each with its own barriers
    int rec_stage_bytes;        // variant 1: offset of the pair box; variant 2: one receptor ring slot (unit)
    int n_rec_stages;           // variant 2: receptor ring depth (units)
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
    const unsigned* n_live;     // optional (device): rotations >= *n_live are dead (device-driven fallback)
    // diagnostics (DOCK_TC_TRACE environment variable; off on the product path):
    // trace = per-role cycle counters summed over CTAs (see TR_*)
    unsigned long long* trace;
};

// trace counters (cycles summed over CTAs)
enum { TR_CTAS = 0, TR_TILES, TR_MMA_TOTAL, TR_MMA_TMEMPTY, TR_MMA_WFULL, TR_MMA_RFULL, TR_EPI_TOTAL, TR_EPI_TMFULL,
       TR_EPI_LDTM, TR_PROD_TOTAL, TR_PROD_WEMPTY, TR_PROD_REMPTY, TR_EPI_WARPS,
       TR_GT_START_NOT = 13,   // max over CTAs of ~(globaltimer at start): ~ = the earliest start (ns)
       TR_GT_END = 14,         // max over CTAs of globaltimer at exit
       TR_GT_CTA_NS = 15,      // sum over CTAs of their lifetime (ns)
       TR_EPI_CHWAIT = 16,     // epilogue / MMA / receptor producer: waits for the next chunk (cycles)
       TR_MMA_CHWAIT = 17,
       TR_REC_CHWAIT = 18,
       TR_EPI_PUB = 19,        // epilogue: publishing lists (cycles)
       TR_EPI_INS = 20,        // epilogue: list insertions, lane gate passes, warp rare-path entries
       TR_EPI_GATE = 21,
       TR_EPI_WRARE = 22,
       TR_CTA0 = 24,           // per CTA (blockIdx.x < TR_MAXCTA): start, end (globaltimer), SM id
       TR_MAXCTA = 1024,
       TR_N = TR_CTA0 + 3 * TR_MAXCTA };
__device__ __forceinline__ unsigned long long gtimer()
{
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}

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

// 32 columns of this warp's TMEM lane quarter; tmem_ld32_nowait leaves the wait::ld to the caller
__device__ __forceinline__ void tmem_ld32_nowait(uint32_t addr, uint32_t (&v)[32])
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
}
__device__ __forceinline__ void tmem_ld_wait() { asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory"); }

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

// ------------------------------------------------------------------ shared epilogue pieces

// One 32-value chunk of scores (rotation of this thread, translations tbase + c0 + j, j < jmax valid)
// into the per-thread exact top-LIST list; GRID writes the chunk to the score grid instead.
// tgk: the unit's global pruning bound T read during the kernel (keys above it can never be among the picks,
// DESIGN.md §8), so (th, th_t) is the smaller of the list's last key and tgk.
template <bool GRID>
__device__ __forceinline__ void epi_chunk(const uint32_t (&v)[32], unsigned long long (&lst)[LIST], float& th,
                                          uint32_t& th_t, uint32_t tbase, int c0, int jmax, float* grid_row,
                                          unsigned* nins = nullptr, unsigned long long tgk = KEY_MAX)
{
    if constexpr (GRID) {
#pragma unroll
        for (int j = 0; j < 32; j++)
            if (j < jmax) grid_row[c0 + j] = __uint_as_float(v[j]);
    } else {
        // fast check: one FMNMX per value; the insertion path is rare after warm-up
        float mn = __uint_as_float(v[0]);
#pragma unroll
        for (int j = 1; j < 32; j++) mn = fminf(mn, __uint_as_float(v[j]));
        // exact gate: a strictly better score, or a tie that could carry a smaller t_lin (exact-zero
        // scores in empty space tie constantly)
        const bool gate = mn < th || (mn == th && tbase + c0 < th_t);
        if (nins) {   // trace: [0] insertions, [1] lane gate passes, [2] warp entries into the rare path
            nins[1] += gate;
            nins[2] += __any_sync(__activemask(), gate) ? 1u : 0u;
        }
        if (gate) {
            // rare path: bitmask of candidates, each extracted with a 5-level select tree (no local memory)
            uint32_t msk = 0;
#pragma unroll
            for (int j = 0; j < 32; j++) msk |= (__uint_as_float(v[j]) <= th && j < jmax) ? (1u << j) : 0u;
            unsigned long long lim = lst[LIST - 1] < tgk ? lst[LIST - 1] : tgk;
            while (msk) {
                const int j = __ffs(msk) - 1;
                msk &= msk - 1;
                const float sv = __uint_as_float(select32(v, j));
                if (sv <= th) {
                    const unsigned long long key = dk::make_key(sv, tbase + c0 + j);
                    if (key < lim) {
                        if (nins) ++nins[0];
                        list_insert(lst, key);
                        lim = lst[LIST - 1] < tgk ? lst[LIST - 1] : tgk;
                        th = dk::key_score_bound(static_cast<uint32_t>(lim >> 32));
                        th_t = static_cast<uint32_t>(lim & 0xffffffffu);
                    }
                }
            }
        }
    }
}

// Item end: bound T_w from k list entries pairwise farther than 2*rho apart, then
// publish bound, mu and the keys <= T (k_merge finishes the greedy).  Loops over the register list
// are fully unrolled (static indices keep it in registers).
// T_w of a list: the key of the k-th entry of a greedy pick from the list with pairwise cyclic Chebyshev distance
// > 2 rho (any k such points bound the true greedy's k-th pick); KEY_MAX if there are fewer.
__device__ __forceinline__ unsigned long long list_bound(const unsigned long long (&lst)[LIST], const TcArgs& a)
{
    unsigned long long Tw = KEY_MAX;
    uint32_t chosen[32];
    int nc = 0;
#pragma unroll
    for (int i = 0; i < LIST; i++) {
        const unsigned long long key = lst[i];
        if (key != KEY_MAX && nc < a.k) {
            const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
            bool far = true;
            for (int c = 0; c < nc; c++) far = far && dk::cheb_cyc(t, chosen[c], a.nx, a.ny, a.nz) > 2 * a.rho;
            if (far) {
                chosen[nc] = t;
                nc++;
                if (nc == a.k) Tw = key;
            }
        }
    }
    return Tw;
}

__device__ __forceinline__ void epi_publish(const unsigned long long (&lst)[LIST], int slot, const TcArgs& a)
{
    unsigned long long Tw = KEY_MAX;
    uint32_t chosen[32];
    int nc = 0;
#pragma unroll
    for (int i = 0; i < LIST; i++) {
        const unsigned long long key = lst[i];
        if (key != KEY_MAX && nc < a.k) {
            const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
            bool far = true;
            for (int c = 0; c < nc; c++) far = far && dk::cheb_cyc(t, chosen[c], a.nx, a.ny, a.nz) > 2 * a.rho;
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

// Epilogue of one tile: Q accumulator rows of NTT translations, TMEM columns [q * NTT, (q + 1) * NTT).
// Warp (quarter, class cls) reads the TMEM lanes of its quarter (lane = rotation); rows are drained in
// order q = 0..Q-1 and each row is released (tm_empty[q]) as soon as the warp's last chunk of it is in
// registers, before that chunk is processed.  Within row q the warp takes the 32-column chunks
// jj = cls, cls + nclass, ... at column ((q + jj) mod NCH) * 32 ("diagonal" classes: over the rows of a
// tile a class's cells are spread like a row class).
// row_full != nullptr: each row has its own "accumulated" barrier (parity row_ph), waited before its drain.
template <int NTT, int Q, bool GRID>
__device__ __forceinline__ void epi_tile(const TcArgs& a, uint32_t tmem, uint64_t* tm_empty, int quarter, int cls,
                                         int nclass, int lane, int slot, bool rot_ok, int tx, int ty, int tz,
                                         unsigned long long (&lst)[LIST], float& th, uint32_t& th_t, bool tr,
                                         long long& tw0, long long& tw1, uint64_t* row_full = nullptr,
                                         unsigned row_ph = 0, unsigned* nins = nullptr, unsigned long long tgk = KEY_MAX)
{
    constexpr int NCH = NTT / 32;
    const int x0 = tx * NTT;
    for (int q = 0; q < Q; q++) {
        if (row_full) {
            twait(&row_full[q], row_ph, tr, tw0);
            tc_fence_after();
        }
        const int y = ty * Q + q, z = tz;
        const bool row_ok = rot_ok && y < a.ny && z < a.nz;
        const uint32_t tbase = static_cast<uint32_t>((z * a.ny + y) * a.nx + x0);
        if (cls >= NCH) {   // no chunk of this row for this class
            __syncwarp();
            if (lane == 0) dk::mbar_arrive(&tm_empty[q]);
            continue;
        }
        if (NCH == 4 && nclass == 2) {
            // two chunks per warp and row: both loads in flight, one wait, release the row, then score --
            // the row is free for the next tile's MMAs before any of its values are processed
            const int c0 = ((q + cls) % NCH) * 32, c1 = ((q + cls + 2) % NCH) * 32;
            uint32_t v0[32], v1[32];
            const long long tl0 = tr ? clock64() : 0;
            const uint32_t base = tmem + (static_cast<uint32_t>(quarter * 32) << 16) + q * NTT;
            tmem_ld32_nowait(base + c0, v0);
            tmem_ld32_nowait(base + c1, v1);
            tmem_ld_wait();
            if (tr) tw1 += clock64() - tl0;
            tc_fence_before();
            __syncwarp();
            if (lane == 0) dk::mbar_arrive(&tm_empty[q]);
            if (!row_ok) continue;
            float* grow = GRID ? a.grid + static_cast<size_t>(slot) * a.nx * a.ny * a.nz + tbase : nullptr;
            epi_chunk<GRID>(v0, lst, th, th_t, tbase, c0, min(32, a.nx - x0 - c0), grow, nins, tgk);
            epi_chunk<GRID>(v1, lst, th, th_t, tbase, c1, min(32, a.nx - x0 - c1), grow, nins, tgk);
            continue;
        }
#pragma unroll 1
        for (int jj = cls; jj < NCH; jj += nclass) {
            const int c0 = ((q + jj) % NCH) * 32;
            uint32_t v[32];
            const long long tl0 = tr ? clock64() : 0;
            tmem_ld32(tmem + (static_cast<uint32_t>(quarter * 32) << 16) + q * NTT + c0, v);
            if (tr) tw1 += clock64() - tl0;
            if (jj + nclass >= NCH) {   // the warp's last chunk of this row is in registers: release the row
                tc_fence_before();
                __syncwarp();
                if (lane == 0) dk::mbar_arrive(&tm_empty[q]);
            }
            if (!row_ok) continue;
            epi_chunk<GRID>(v, lst, th, th_t, tbase, c0, min(32, a.nx - x0 - c0),
                            GRID ? a.grid + static_cast<size_t>(slot) * a.nx * a.ny * a.nz + tbase : nullptr, nullptr,
                            tgk);
        }
    }
}

// Shared-memory box geometry of the PAIR scheme (must match make_tc_plan): x extent of the (hi,lo) box
// and of the (hi(x),hi(x+1)) box for NTT translations per row.
__host__ __device__ constexpr int pair_txb(int m, int ntt = NT)
{
    return (ntt + (m + 1) / 2 * 2 - 1) > (4 * ((m + 3) / 4) + ntt - 2) ? (ntt + (m + 1) / 2 * 2 - 1)
                                                                       : (4 * ((m + 3) / 4) + ntt - 2);
}
// Variant 1 sizes each box to what its pass reads: main (hi,lo) box x extent NT + 2*MXP - 1, pair box
// NT + 4*MXQ - 2 (slot x already holds voxel x + 1) -- at m = 4 the 448 B saved let a 7th weight stage fit.
__host__ __device__ constexpr int main_box_txb(int m) { return NT + (m + 1) / 2 * 2 - 1; }
__host__ __device__ constexpr int pair_box_txb(int m) { return NT + 4 * ((m + 3) / 4) - 2; }
// compile-time loop: f(std::integral_constant<int, i>) for i in [0, N)
template <class F, int... I>
__device__ __forceinline__ void static_for_impl(F&& f, std::integer_sequence<int, I...>)
{
    (f(std::integral_constant<int, I>{}), ...);
}
template <int N, class F>
__device__ __forceinline__ void static_for(F&& f)
{
    static_for_impl(f, std::make_integer_sequence<int, N>{});
}

// Byte offset of K-step s inside the PAIR pass-1 box ((hi,lo) voxels, 2 per K-step) and pass-2 box
// ((hi(x),hi(x+1)) slots, 4 voxels per K-step); padding steps (zero weights) re-read the last real
// step's voxels.
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

// ------------------------------------------------------------------ variant 1: resident receptor boxes
//
// One channel group (P <= 4), PAIR scheme: pass 1 reads the (hi, lo) receptor box -> Rhi*Whi + Rlo*Whi
// over 2 voxels per MMA; pass 2 reads a second box whose 16-B slot x holds (Rhi(x), Rhi(x+1)), so one
// K = 16 MMA covers 4 voxels of Rhi*Wlo (chunk LBO = 32 B): 3 MMAs per 4 voxels instead of 4.  Both
// whole boxes (all m z-planes, Q = 4 rows + halo) are resident; the main box is released after pass 1
// and the pair box after pass 2, so one buffer of each gives full TMA/MMA overlap.  One TMEM buffer of
// Q x 128 columns; rows are released one by one by the epilogue and restarted in that order.
// Occupancy schedule: a ring stage (KS K-steps) whose weights are zero for all 128 rotations of the block would
// add exact zeros to every accumulator; the block's stage mask (k_tc_block_tables) skips it, and the weight
// stream holds only the block's active stages.  The schedule stays fully unrolled (immediate receptor offsets).
template <int M, bool GRID>
__global__ void __launch_bounds__(NTHREADS, 1) k_corr_tc(const __grid_constant__ CUtensorMap tmap,
                                                          const __grid_constant__ CUtensorMap tmap_pair,
                                                          const __grid_constant__ CUtensorMap tmap_b, const TcArgs a)
{
    constexpr int Q = 4;
    constexpr int KS = KSTEPS;                 // K-steps per weight-ring stage (one wait/commit per KS steps)
    constexpr unsigned STAGE = KS * WCHUNK;
    constexpr int MXP = (M + 1) / 2, MXQ = (M + 3) / 4;
    constexpr int S1 = M * M * MXP, S1P = (S1 + KS - 1) / KS * KS;
    constexpr int S2 = M * M * MXQ, S2P = (S2 + KS - 1) / KS * KS;
    constexpr int NSTEPS = S1P + S2P;
    constexpr uint32_t ROW16 = static_cast<uint32_t>(main_box_txb(M)) * 16u;    // main box row pitch
    constexpr uint32_t ROWTY = static_cast<uint32_t>(Q + M - 1) * ROW16;
    constexpr uint32_t ROW16P = static_cast<uint32_t>(pair_box_txb(M)) * 16u;   // pair box row pitch
    constexpr uint32_t ROWTYP = static_cast<uint32_t>(Q + M - 1) * ROW16P;
    // main half-boxes: A = z planes [0, MH) at 0, B = [MH, M) at OFFB (128-B aligned for TMA); pass-1 K-steps
    // from KB on read B, so B is needed from stage SB on and A is done after stage SA
    constexpr int MH = (M + 1) / 2;
    constexpr uint32_t OFFB = (MH * ROWTY + 127u) / 128u * 128u, GAPB = OFFB - MH * ROWTY;
    constexpr int KB = MH * MXP * M, SB = KB / KS, SA = (KB - 1) / KS;
    constexpr bool HAS_B = M > MH;
    static_assert(Q * NT <= 512, "TMEM has 512 columns");
    extern __shared__ __align__(128) unsigned char smem[];   // TMA destinations: 128 B; no-swizzle UMMA operands: 16 B
    constexpr int NCR = 4;                     // chunk ring: the weight producer posts, the other roles take
    __shared__ uint64_t bars[2 * 3 + 2 * WSTAGES + 2 * Q + 2 * NCR];
    __shared__ uint32_t tmem_base_s;
    __shared__ long long s_cg[NCR];            // chunk: first (block, tile) pair g = block * ntiles + tile
    __shared__ int s_cn[NCR];                  // chunk: tiles (0 = no more work)
    uint64_t* rec_full = bars;        // [3]: main half-box A, pair box, main half-box B
    uint64_t* rec_empty = bars + 3;
    uint64_t* w_full = bars + 6;
    uint64_t* w_empty = w_full + WSTAGES;
    uint64_t* tm_full = w_empty + WSTAGES;   // [Q]: row q accumulated (the staircase finishes rows one by one)
    uint64_t* tm_empty = tm_full + Q;        // [Q]: row q drained, so the next tile restarts row by row
    uint64_t* ch_full = tm_empty + Q;        // [NCR]: chunk posted
    uint64_t* ch_empty = ch_full + NCR;      // [NCR]: chunk taken by the MMA, receptor and epilogue roles

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int n_eff = a.n_live ? min(a.n_slots, static_cast<int>(*a.n_live)) : a.n_slots;
    const long long live_blocks = a.n_blocks > 0 ? a.n_blocks : (n_eff + ROT - 1) / ROT;
    // block of the call's block order for a local block index (block sharding: this rank's blocks only)
    auto gblock = [&](long long lb) -> long long { return a.blkmap ? a.blkmap[lb] : lb; };
    // Work: a sequence of chunks (g, n) = n consecutive tiles of one rotation block starting at the (block,
    // tile) pair g = block * ntiles + tile.  Region mode: the one chunk (block, region) of this CTA.  Dynamic
    // mode: chunk c = (block c / cpb, tiles [(c % cpb) chunk, ..)), c in [0, n_chunks), split into NS
    // segments with one counter each.  A CTA takes the chunks of its own segment in order (a contiguous
    // tile range of one block, so its top-k lists live long: a list restart costs a burst of insertions),
    // then helps the next segments that still have chunks: CTAs whose tiles are cheaper (per-tile cost
    // varies with the receptor region through the epilogue's insertions) take more.  The NS = S =
    // gridDim.x segments are contiguous ranges of the chunk space, so concurrent CTAs read the receptor at
    // scattered positions: that costs L2 misses (~2.2 GB of DRAM reads per prod launch instead of ~0.1)
    // but spreads the reads over the L2 slices; region-major segments that keep the CTAs in step on a few
    // receptor windows cut DRAM to 0.1 GB and ran 13 % slower (hot L2 lines).
    const int cpb = a.chunk > 0 ? (a.ntiles + a.chunk - 1) / a.chunk : 0;
    const long long n_chunks = live_blocks * cpb;
    const int S = gridDim.x;
    const int NS = S;
    long long reg_g = 0;
    int reg_n = 0;
    if (a.chunk <= 0) {
        const int block = blockIdx.x / a.G, region = blockIdx.x % a.G;
        const int tile_begin = region * a.tiles_per_region;
        if (block < live_blocks && tile_begin < a.ntiles) {
            reg_g = static_cast<long long>(block) * a.ntiles + tile_begin;
            reg_n = min(a.ntiles, tile_begin + a.tiles_per_region) - tile_begin;
        }
    }
    if (a.chunk > 0 ? n_chunks == 0 : reg_n == 0) {
        // uniform: no work (no live rotations in the device-driven fallback, or an empty region)
        if (a.chunk > 0 && threadIdx.x == 0 && atomicAdd(&a.sched[0], 1ull) == static_cast<unsigned>(S - 1))
            for (int j = 0; j <= NS; j++) a.sched[j] = 0;
        return;
    }
    unsigned char* rec_smem = smem;   // [main box | pair box at a.rec_stage_bytes]
    unsigned char* w_smem = smem + a.rec_stage_bytes + ((a.box_bytes_pair + 127) & ~127);

    if (threadIdx.x == 0) {
        for (int i = 0; i < 3; i++) {
            dk::mbar_init(&rec_full[i], 1);
            dk::mbar_init(&rec_empty[i], 1);
        }
        for (int i = 0; i < a.wstages; i++) {
            dk::mbar_init(&w_full[i], 1);
            dk::mbar_init(&w_empty[i], 1);
        }
        for (int i = 0; i < Q; i++) {
            dk::mbar_init(&tm_full[i], 1);
            dk::mbar_init(&tm_empty[i], a.nepi);
        }
        for (int i = 0; i < NCR; i++) {
            dk::mbar_init(&ch_full[i], 1);
            dk::mbar_init(&ch_empty[i], 2 + a.nepi);
        }
        dk::fence_mbar_init();
    }
    if (warp == 1) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(
            dk::smem_u32(&tmem_base_s)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    const uint32_t tmem = tmem_base_s;

    const bool tr = a.trace != nullptr;
    long long tw0 = 0, tw1 = 0, tw2 = 0, tstart = tr ? clock64() : 0;   // per-role trace accumulators
    const unsigned long long gt0 = tr ? gtimer() : 0;
    int cs = 0;             // chunk ring slot / phase of this role
    unsigned cph = 0;
    // consumer side of the chunk ring (one thread per role; the epilogue warps each arrive once)
    long long tch = 0;      // chunk-wait cycles of this role (trace)
    auto take_chunk = [&](long long& g, bool arrive) -> int {
        twait(&ch_full[cs], cph, tr, tch);
        g = s_cg[cs];
        const int n = s_cn[cs];
        if (arrive) dk::mbar_arrive(&ch_empty[cs]);
        if (++cs == NCR) {
            cs = 0;
            cph ^= 1u;
        }
        return n;
    };
    int n_tiles = 0;        // tiles this CTA processed (trace)
    {
        if (warp == 0) {
            // ------------------------------------------------ weight producer (one thread): the whole A
            // stream in stage order; it never waits on a receptor buffer (warp 2 + nepi loads those)
            // (warp-wide: lane 0 streams, all lanes search for chunks to help with)
            // segment j: chunk ids [lo, hi)
            auto seg_range = [&](int j, long long& lo, long long& hi) {
                if (a.seg) {
                    lo = a.seg[j];
                    hi = a.seg[j + 1];
                } else {
                    lo = static_cast<long long>(j) * n_chunks / NS;
                    hi = static_cast<long long>(j + 1) * n_chunks / NS;
                }
            };
            int seg = blockIdx.x;
            auto fetch = [&]() -> long long {   // next chunk id, -1 when every segment is exhausted
                for (;;) {
                    long long c = -1;
                    if (lane == 0) {
                        long long lo, hi;
                        seg_range(seg, lo, hi);
                        const long long t = static_cast<long long>(atomicAdd(&a.sched[1 + seg], 1ull));
                        if (lo + t < hi) c = lo + t;
                    }
                    c = __shfl_sync(0xffffffffu, c, 0);
                    if (c >= 0) return c;
                    int found = -1;
                    for (int base = 1; base < NS && found < 0; base += 32) {
                        bool has = false;
                        if (base + lane < NS) {
                            const int j = (seg + base + lane) % NS;
                            long long lo, hi;
                            seg_range(j, lo, hi);
                            const unsigned long long t = *reinterpret_cast<volatile unsigned long long*>(&a.sched[1 + j]);
                            has = lo + static_cast<long long>(t) < hi;
                        }
                        const unsigned mk = __ballot_sync(0xffffffffu, has);
                        if (mk) found = (seg + base + __ffs(mk) - 1) % NS;
                    }
                    if (found < 0) return -1;
                    seg = found;
                }
            };
            int ws = 0, wph = 0, wuse = 0;
            long long c = a.chunk > 0 ? fetch() : 0;   // dynamic mode: the chunk to post next
            for (bool first = true;; first = false) {
                long long g = 0;
                int n = 0;
                if (a.chunk > 0) {
                    if (c >= 0) {
                        const long long blk = c / cpb;
                        const int t0 = static_cast<int>(c % cpb) * a.chunk;
                        g = blk * a.ntiles + t0;
                        n = min(a.chunk, a.ntiles - t0);
                    }
                } else if (first) {
                    g = reg_g;
                    n = reg_n;
                }
                // post the chunk (the slot is free once all consumers took the chunk NCR posts ago)
                if (lane == 0) {
                    dk::mbar_wait(&ch_empty[cs], cph ^ 1u);
                    s_cg[cs] = g;
                    s_cn[cs] = n;
                    dk::mbar_arrive(&ch_full[cs]);
                }
                __syncwarp();
                if (++cs == NCR) {
                    cs = 0;
                    cph ^= 1u;
                }
                if (n == 0) break;
                if (a.chunk > 0) c = fetch();   // one chunk of lookahead: the atomic hides behind the stream
                n_tiles += n;
                if (lane == 0) {
                    const long long blk = gblock(g / a.ntiles);
                    const unsigned char* wsrc = a.W + static_cast<size_t>(blk) * NSTEPS * WCHUNK;
                    const int nst = a.kinfo[blk].x;   // the block's active stages (compacted weight stream)
                    for (int ti = 0; ti < n; ti++) {
                        for (int st = 0; st < nst; st++) {
                            if (wuse >= a.wstages) twait(&w_empty[ws], wph ^ 1, tr, tw0);
                            dk::mbar_arrive_expect_tx(&w_full[ws], STAGE);
                            dk::bulk_load(w_smem + static_cast<size_t>(ws) * STAGE,
                                          wsrc + static_cast<size_t>(st) * STAGE, STAGE, &w_full[ws]);
                            wuse++;
                            if (++ws == a.wstages) {
                                ws = 0;
                                wph ^= 1;
                            }
                        }
                    }
                }
                __syncwarp();
            }
            if (tr && lane == 0) {
                atomicAdd(&a.trace[TR_PROD_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                atomicAdd(&a.trace[TR_PROD_WEMPTY], static_cast<unsigned long long>(tw0));
                atomicAdd(&a.trace[TR_CTAS], 1ull);
                atomicAdd(&a.trace[TR_TILES], static_cast<unsigned long long>(n_tiles));
            }
            __syncwarp();
        } else if (warp == 2 + a.nepi) {
            // ------------------------------------------------ receptor producer (one thread): main box of
            // tile t as soon as pass 1 of t-1 released it, pair box as soon as pass 2 of t-1 did
            if (elect_one()) {
                dk::prefetch_tmap(&tmap);
                dk::prefetch_tmap(&tmap_pair);
                dk::prefetch_tmap(&tmap_b);
                int ti = 0;   // tiles so far (buffer phases)
                long long g;
                for (int n; (n = take_chunk(g, true)) > 0;) {
                    const int t0 = static_cast<int>(g % a.ntiles);
                    int tx = t0 % a.ntx, ty = (t0 / a.ntx) % a.nty, tz = t0 / (a.ntx * a.nty);
                    for (int j = 0; j < n; j++, ti++) {
                        // in the order the MMAs need them: half-box A, half-box B, pair box
                        for (int k = 0; k < 3; k++) {
                            const int which = k == 0 ? 0 : k == 1 ? 2 : 1;
                            if (which == 2 && !HAS_B) continue;
                            if (ti > 0) twait(&rec_empty[which], (ti - 1) & 1, tr, tw1);
                            dk::mbar_arrive_expect_tx(&rec_full[which], which == 0   ? a.box_bytes
                                                                        : which == 2 ? a.box_bytes_b
                                                                                     : a.box_bytes_pair);
                            tma_load_5d(rec_smem + (which == 0 ? 0 : which == 2 ? a.rec_off_b : a.rec_stage_bytes),
                                        which == 0 ? &tmap : which == 2 ? &tmap_b : &tmap_pair, 0, tx * NT, ty * Q,
                                        tz + (which == 2 ? MH : 0), 0, &rec_full[which]);
                        }
                        if (++tx == a.ntx) {
                            tx = 0;
                            if (++ty == a.nty) {
                                ty = 0;
                                tz++;
                            }
                        }
                    }
                }
                if (tr) {
                    atomicAdd(&a.trace[TR_PROD_REMPTY], static_cast<unsigned long long>(tw1));
                    atomicAdd(&a.trace[TR_REC_CHWAIT], static_cast<unsigned long long>(tch));
                }
            }
            __syncwarp();
        } else if (warp == 1) {
            // ------------------------------------------------ MMA issuer (one thread runs the whole schedule)
            // The stage loops are unrolled so every descriptor offset is an immediate and the tcgen05 queue
            // stays fed (issuing per K-step from a converged warp capped the tensor pipe at 40-47 %).
            // Staircase: the first D and the last D weight stages of a tile are issued row by row, so row q
            // finishes (tm_full[q]) while rows q+1.. still compute and restarts as soon as the epilogue has
            // drained it -- the TMEM drain (64 B/clk, a third of the MMA time at m = 4) overlaps the MMAs
            // instead of stalling the tensor pipe at every tile boundary.
            constexpr uint32_t idesc = umma_idesc(ROT, NT);
            constexpr int NS1 = S1P / KS, NS2 = S2P / KS;
            constexpr int DS = DOCK_TC_STAIR;
            constexpr int D = NS1 < NS2 ? (NS1 < DS ? NS1 : DS) : (NS2 < DS ? NS2 : DS);   // staircase depth
            const uint32_t rec0 = dk::smem_u32(rec_smem), w0 = dk::smem_u32(w_smem);
            const uint64_t dA0 = umma_desc(w0, ROT * 16, 128);                 // + (slot offset >> 4)
            const uint64_t dB0 = umma_desc(rec0, 16, 128);                     // + (voxel offset >> 4)
            const uint64_t dP0 = umma_desc(rec0 + a.rec_stage_bytes, 32, 128);
            // byte offset of pass-1 K-step s: z planes from MH on sit in half-box B, GAPB further on
            constexpr auto off1 = [](int s) constexpr -> uint32_t {
                const int t = s < S1 ? s : S1 - 1;
                return pair_off1(M, s, ROW16, ROWTY) + (t / (MXP * M) >= MH ? GAPB : 0u);
            };
            if (elect_one()) {
                uint32_t ws = 0, wph = 0;   // ring slot / phase of the next stage
                const uint32_t nws = static_cast<uint32_t>(a.wstages);
                // slot and phase of the stage `ahead` stages after the next one
                auto slot_of = [&](int ahead, uint32_t& ph) -> uint32_t {
                    uint32_t sl = ws + static_cast<uint32_t>(ahead);
                    ph = wph;
                    if (sl >= nws) {
                        sl -= nws;
                        ph ^= 1u;
                    }
                    return sl;
                };
                auto advance = [&](int n) {
                    for (int i = 0; i < n; i++)
                        if (++ws == nws) {
                            ws = 0;
                            wph ^= 1;
                        }
                };
                int ti = 0;   // tiles so far (buffer phases)
                long long g, mblk = -1;
                unsigned long long smk = ~0ull;   // the block's active stages: bit st = dense stage st
                constexpr int NSTG = NS1 + NS2;
                constexpr bool MASKED = NSTG <= 64;   // stage masks are one 64-bit word (m <= 6); else dense
                constexpr unsigned long long HEADM = (1ull << D) - 1ull;
                // stage st active / active stages before st (dense when unmasked)
                auto act = [&](int st) -> bool { return !MASKED || ((smk >> (st & 63)) & 1ull); };
                auto below = [&](unsigned long long mk, int st) -> int {
                    return MASKED ? __popcll(mk & ((1ull << (st & 63)) - 1ull)) : st;
                };
                for (int n; (n = take_chunk(g, true)) > 0;) {
                    const long long blk = gblock(g / a.ntiles);
                    if (MASKED && blk != mblk) {
                        const int4 inf = a.kinfo[blk];
                        smk = static_cast<unsigned long long>(static_cast<uint32_t>(inf.z)) |
                              (static_cast<unsigned long long>(static_cast<uint32_t>(inf.w)) << 32);
                        mblk = blk;
                    }
                    const int nh = MASKED ? __popcll(smk & HEADM) : D;                 // active head stages
                    const unsigned long long tmk = MASKED ? smk >> ((NSTG - D) & 63) : ~0ull;   // tail stages
                    const int nt = MASKED ? __popcll(tmk & HEADM) : D;
                for (int j = 0; j < n; j++, ti++) {
                    twait(&rec_full[0], ti & 1, tr, tw2);
                    tc_fence_after();
                    if constexpr (HAS_B && SB < D) {   // the head reads half-box B too
                        twait(&rec_full[2], ti & 1, tr, tw2);
                        tc_fence_after();
                    }
                    // pass 1, stages [0, D): row by row, each row after the epilogue released it
#pragma unroll
                    for (int q = 0; q < Q; q++) {
                        if (ti > 0) {
                            twait(&tm_empty[q], (ti - 1) & 1, tr, tw0);
                            tc_fence_after();
                        }
#pragma unroll
                        for (int st = 0; st < D; st++) {
                            if (!act(st)) continue;
                            const int rk = below(smk, st);   // ring stages before it
                            uint32_t ph;
                            const uint32_t sl = slot_of(rk, ph);
                            if (q == 0) {
                                twait(&w_full[sl], ph, tr, tw1);
                                tc_fence_after();
                            }
                            const uint64_t da0 = dA0 + ((sl * STAGE) >> 4);
#pragma unroll
                            for (int ks = 0; ks < KS; ks++)
                                umma_bf16(tmem + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                          dB0 + ((off1(st * KS + ks) + q * ROW16) >> 4), idesc,
                                          (rk == 0 && ks == 0) ? 0u : 1u);
                        }
                    }
                    for (int i = 0; i < nh; i++) {
                        uint32_t ph;
                        umma_commit(&w_empty[slot_of(i, ph)]);
                    }
                    advance(nh);
                    if constexpr (SA < D) umma_commit(&rec_empty[0]);   // half-box A done with the head
                    int nact = nh;   // active stages issued so far in this tile (0: the next one overwrites)
                    // pass 1, stages [D, NS1): all rows per stage
#pragma unroll
                    for (int st = D; st < NS1; st++) {
                        if (HAS_B && SB >= D && st == SB) {   // the first stage that reads half-box B
                            twait(&rec_full[2], ti & 1, tr, tw2);
                            tc_fence_after();
                        }
                        if (!act(st)) {
                            if (SA >= D && st == SA) umma_commit(&rec_empty[0]);
                            continue;
                        }
                        twait(&w_full[ws], wph, tr, tw1);
                        tc_fence_after();
                        const uint64_t da0 = dA0 + ((ws * STAGE) >> 4);
                        const uint32_t acc0 = nact == 0 ? 0u : 1u;
#pragma unroll
                        for (int ks = 0; ks < KS; ks++)
#pragma unroll
                            for (int q = 0; q < Q; q++)
                                umma_bf16(tmem + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                          dB0 + ((off1(st * KS + ks) + q * ROW16) >> 4), idesc,
                                          ks == 0 ? acc0 : 1u);
                        umma_commit(&w_empty[ws]);
                        advance(1);
                        nact++;
                        if (SA >= D && st == SA) umma_commit(&rec_empty[0]);   // half-box A done
                    }
                    if constexpr (HAS_B) umma_commit(&rec_empty[2]);
                    twait(&rec_full[1], ti & 1, tr, tw2);
                    tc_fence_after();
                    // pass 2, stages [0, NS2 - D): all rows per stage
#pragma unroll
                    for (int st = 0; st < NS2 - D; st++) {
                        if (!act(NS1 + st)) continue;
                        twait(&w_full[ws], wph, tr, tw1);
                        tc_fence_after();
                        const uint64_t da0 = dA0 + ((ws * STAGE) >> 4);
                        const uint32_t acc0 = nact == 0 ? 0u : 1u;
#pragma unroll
                        for (int ks = 0; ks < KS; ks++)
#pragma unroll
                            for (int q = 0; q < Q; q++)
                                umma_bf16(tmem + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                          dP0 + ((pair_off2(M, st * KS + ks, ROW16P, ROWTYP) + q * ROW16P) >> 4), idesc,
                                          ks == 0 ? acc0 : 1u);
                        umma_commit(&w_empty[ws]);
                        advance(1);
                        nact++;
                    }
                    // pass 2, stages [NS2 - D, NS2): row by row; row q is complete after its block
#pragma unroll
                    for (int q = 0; q < Q; q++) {
#pragma unroll
                        for (int j = 0; j < D; j++) {
                            if (MASKED && !((tmk >> j) & 1ull)) continue;
                            const int st = NS2 - D + j;
                            const int rk = below(tmk, j);
                            uint32_t ph;
                            const uint32_t sl = slot_of(rk, ph);
                            if (q == 0) {
                                twait(&w_full[sl], ph, tr, tw1);
                                tc_fence_after();
                            }
                            const uint64_t da0 = dA0 + ((sl * STAGE) >> 4);
#pragma unroll
                            for (int ks = 0; ks < KS; ks++)
                                umma_bf16(tmem + q * NT, da0 + ((ks * WCHUNK) >> 4),
                                          dP0 + ((pair_off2(M, st * KS + ks, ROW16P, ROWTYP) + q * ROW16P) >> 4), idesc,
                                          (nact + rk == 0 && ks == 0) ? 0u : 1u);
                        }
                        umma_commit(&tm_full[q]);
                    }
                    for (int i = 0; i < nt; i++) {
                        uint32_t ph;
                        umma_commit(&w_empty[slot_of(i, ph)]);
                    }
                    advance(nt);
                    umma_commit(&rec_empty[1]);
                }
                }
                if (tr) {
                    atomicAdd(&a.trace[TR_MMA_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                    atomicAdd(&a.trace[TR_MMA_TMEMPTY], static_cast<unsigned long long>(tw0));
                    atomicAdd(&a.trace[TR_MMA_WFULL], static_cast<unsigned long long>(tw1));
                    atomicAdd(&a.trace[TR_MMA_RFULL], static_cast<unsigned long long>(tw2));
                    atomicAdd(&a.trace[TR_MMA_CHWAIT], static_cast<unsigned long long>(tch));
                }
            }
            __syncwarp();
        } else {
            // ------------------------------------------------ epilogue warps
            const int quarter = warp & 3;
            const int cls = (warp - 2) >> 2;
            const int nclass = a.nepi >> 2;
            const int r = quarter * 32 + lane;                  // rotation within the block (TMEM lane)
            long long cur = -1;                                 // rotation block of the lists
            int slot = 0;
            bool rot_ok = false;
            unsigned long long lst[LIST];
#pragma unroll
            for (int i = 0; i < LIST; i++) lst[i] = KEY_MAX;
            float th = __int_as_float(0x7f800000);   // score of the gate key: min(list's last key, tgk) (+inf: none)
            uint32_t th_t = 0xffffffffu;             // t_lin of the gate key
            unsigned long long tgk = KEY_MAX;        // the unit's pruning bound T as last read
            int since = 0;                            // tiles of the current block (periodic bound publish)
            int ti = 0;                               // tiles so far (TMEM phases)
            long long g, tpub = 0;
            unsigned nins[3] = {0, 0, 0};
            for (int n; (n = take_chunk(g, false)) > 0;) {
                __syncwarp();
                if (lane == 0) dk::mbar_arrive(&ch_empty[(cs + NCR - 1) % NCR]);
                const long long blk = g / a.ntiles;
                if (blk != cur) {
                    // a new rotation block: publish the lists of the previous one (once: the chunk sequence
                    // of a CTA is increasing, so it never returns to a block)
                    if constexpr (!GRID) {
                        const long long tp0 = tr ? clock64() : 0;
                        if (cur >= 0 && rot_ok) epi_publish(lst, slot, a);
                        if (tr) tpub += clock64() - tp0;
                    }
#pragma unroll
                    for (int i = 0; i < LIST; i++) lst[i] = KEY_MAX;
                    th = __int_as_float(0x7f800000);
                    th_t = 0xffffffffu;
                    tgk = KEY_MAX;
                    since = 0;
                    cur = blk;
                    const int pos = static_cast<int>(gblock(blk)) * ROT + r;   // position in the block order
                    rot_ok = pos < n_eff;
                    slot = (a.perm && rot_ok) ? a.perm[pos] : pos;     // the unit it holds
                }
                const int t0 = static_cast<int>(g % a.ntiles);
                int tx = t0 % a.ntx, ty = (t0 / a.ntx) % a.nty, tz = t0 / (a.ntx * a.nty);
                for (int j = 0; j < n; j++, ti++) {
                    if (!GRID && rot_ok) {
                        // the unit's pruning bound T so far (other lists' published T_w): keys above it cannot be
                        // picks, so the gate also skips them (fewer insertions; DESIGN.md §8 stays exact)
                        const unsigned long long tg = *reinterpret_cast<volatile unsigned long long*>(&a.T[slot]);
                        if (tg < tgk) {
                            tgk = tg;
                            const unsigned long long lim = lst[LIST - 1] < tgk ? lst[LIST - 1] : tgk;
                            th = dk::key_score_bound(static_cast<uint32_t>(lim >> 32));
                            th_t = static_cast<uint32_t>(lim & 0xffffffffu);
                        }
                        if ((++since & 31) == 0) {   // publish this list's bound every 32 tiles
                            const unsigned long long tw = list_bound(lst, a);
                            if (tw < tgk) atomicMin(&a.T[slot], tw);
                        }
                    }
                    epi_tile<NT, Q, GRID>(a, tmem, tm_empty, quarter, cls, nclass, lane, slot, rot_ok, tx, ty, tz, lst,
                                          th, th_t, tr, tw0, tw1, tm_full, ti & 1, tr ? nins : nullptr, tgk);
                    if (++tx == a.ntx) {
                        tx = 0;
                        if (++ty == a.nty) {
                            ty = 0;
                            tz++;
                        }
                    }
                }
            }
            __syncwarp();
            if (lane == 0) dk::mbar_arrive(&ch_empty[(cs + NCR - 1) % NCR]);   // the end marker
            if (tr && lane == 0) {
                atomicAdd(&a.trace[TR_EPI_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                atomicAdd(&a.trace[TR_EPI_TMFULL], static_cast<unsigned long long>(tw0));
                atomicAdd(&a.trace[TR_EPI_LDTM], static_cast<unsigned long long>(tw1));
                atomicAdd(&a.trace[TR_EPI_WARPS], 1ull);
                atomicAdd(&a.trace[TR_EPI_CHWAIT], static_cast<unsigned long long>(tch));
                atomicAdd(&a.trace[TR_EPI_PUB], static_cast<unsigned long long>(tpub));
            }
            if (tr) {
                atomicAdd(&a.trace[TR_EPI_INS], static_cast<unsigned long long>(nins[0]));
                atomicAdd(&a.trace[TR_EPI_GATE], static_cast<unsigned long long>(nins[1]));
                if (lane == 0) atomicAdd(&a.trace[TR_EPI_WRARE], static_cast<unsigned long long>(nins[2]));
            }
            if constexpr (!GRID) {
                if (cur >= 0 && rot_ok) epi_publish(lst, slot, a);
            }
        }
    }
    tc_fence_before();
    __syncthreads();
    if (warp == 1) asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
    // dynamic mode: the last CTA to finish (every fetch of every CTA is done by then) resets the counters
    if (a.chunk > 0 && threadIdx.x == 0 && atomicAdd(&a.sched[0], 1ull) == static_cast<unsigned>(S - 1))
        for (int j = 0; j <= NS; j++) a.sched[j] = 0;
    if (tr && threadIdx.x == 0) {
        const unsigned long long gt1 = gtimer();
        atomicMax(&a.trace[TR_GT_START_NOT], ~gt0);
        atomicMax(&a.trace[TR_GT_END], gt1);
        atomicAdd(&a.trace[TR_GT_CTA_NS], gt1 - gt0);
        if (blockIdx.x < TR_MAXCTA) {
            unsigned smid;
            asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
            a.trace[TR_CTA0 + 3 * blockIdx.x] = gt0;
            a.trace[TR_CTA0 + 3 * blockIdx.x + 1] = gt1;
            a.trace[TR_CTA0 + 3 * blockIdx.x + 2] = smid;
        }
    }
}

// ------------------------------------------------------------------ variant 2: streamed receptor planes
//
// Any number of channel groups G (P <= 32) and any probe size m <= 8, PAIR scheme per group, NTT
// translations per MMA row (NTT = 64, 128 or 160 chosen at init to fit nx with the least waste) and Q
// rows per tile (Q * NTT <= 512 TMEM columns).  K is walked unit by unit, unit u = (g, vz): the main
// z-plane box of group g ((hi, lo) voxels, pass 1, M * MXP K-steps over (vy, vxp)) and its pair z-plane
// box ((hi(x), hi(x+1)) slots, pass 2, M * MXQ K-steps over (vy, vxq)), padded to whole ring stages.
// The two planes of a unit share one slot of an NR-deep receptor ring (one TMA box each, one barrier
// pair per slot), so shared memory holds NR units whatever G and m are -- this is what lets the
// large configuration (P = 22, m = 8) run on the tensor cores.
__host__ __device__ constexpr int unit_ksteps(int m) { return m * ((m + 1) / 2) + m * ((m + 3) / 4); }
__host__ __device__ constexpr int unit_ksteps_padded(int m) { return (unit_ksteps(m) + KSTEPS - 1) / KSTEPS * KSTEPS; }
__host__ __device__ constexpr uint32_t stream_plane_stride(int m, int ntt, int q)
{
    return (static_cast<uint32_t>(q + m - 1) * static_cast<uint32_t>(pair_txb(m, ntt)) * 16u + 127u) / 128u * 128u;
}
// byte offset of K-step s of a unit inside its slot (main plane at 0, pair plane at pstride)
__host__ __device__ constexpr uint32_t unit_off(int m, int s, uint32_t row16, uint32_t pstride)
{
    const int mxp = (m + 1) / 2, mxq = (m + 3) / 4, kp1 = m * mxp, kp2 = m * mxq;
    return s < kp1        ? static_cast<uint32_t>(s / mxp) * row16 + static_cast<uint32_t>(s % mxp) * 32u
           : s < kp1 + kp2 ? pstride + static_cast<uint32_t>((s - kp1) / mxq) * row16 +
                                static_cast<uint32_t>((s - kp1) % mxq) * 64u
                          : 0u;   // padding step: zero weights, any finite receptor data
}

template <int M, int NTT, int Q, bool GRID>
__global__ void __launch_bounds__(NTHREADS, 1) k_corr_tcs(const __grid_constant__ CUtensorMap tmap,
                                                           const __grid_constant__ CUtensorMap tmap_pair,
                                                           const TcArgs a)
{
    constexpr int KS = KSTEPS;
    constexpr unsigned STAGE = KS * WCHUNK;
    constexpr int MXP = (M + 1) / 2;
    constexpr int KP1 = M * MXP;                  // pass-1 K-steps of a unit
    constexpr int KU = unit_ksteps(M);
    constexpr int KUP = unit_ksteps_padded(M);
    constexpr int NSU = KUP / KS;                 // weight stages per unit
    constexpr uint32_t ROW16 = static_cast<uint32_t>(pair_txb(M, NTT)) * 16u;
    constexpr uint32_t PLANE = static_cast<uint32_t>(Q + M - 1) * ROW16;   // bytes of one z-plane box
    constexpr uint32_t PSTRIDE = stream_plane_stride(M, NTT, Q);
    constexpr int NRMAX = 4;
    static_assert(Q * NTT <= 512, "TMEM has 512 columns");
    static_assert(NTT % 32 == 0 && NTT >= 32 && NTT <= 256, "MMA N");
    extern __shared__ __align__(128) unsigned char smem[];   // TMA destinations: 128 B; no-swizzle UMMA operands: 16 B
    __shared__ uint64_t bars[2 * NRMAX + 2 * WSTAGES + 1 + Q];
    __shared__ uint32_t tmem_base_s;
    uint64_t* rec_full = bars;
    uint64_t* rec_empty = bars + NRMAX;
    uint64_t* w_full = bars + 2 * NRMAX;
    uint64_t* w_empty = w_full + WSTAGES;
    uint64_t* tm_full = w_empty + WSTAGES;
    uint64_t* tm_empty = tm_full + 1;   // [Q]

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int block = blockIdx.x / a.G, region = blockIdx.x % a.G;
    const int n_eff = a.n_live ? min(a.n_slots, static_cast<int>(*a.n_live)) : a.n_slots;
    if (block * ROT >= n_eff) return;   // uniform: a dead block of the device-driven fallback
    const int tile_begin = region * a.tiles_per_region;
    const int tile_end = min(a.ntiles, tile_begin + a.tiles_per_region);
    const int n_tiles = tile_end - tile_begin;
    const int NU = a.G_ch * M;          // units per tile
    const int NR = a.n_rec_stages;      // receptor ring depth (units)
    unsigned char* rec_smem = smem;     // [NR][slot = main plane | pair plane]
    unsigned char* w_smem = smem + NR * a.rec_stage_bytes;

    if (threadIdx.x == 0) {
        for (int i = 0; i < NR; i++) {
            dk::mbar_init(&rec_full[i], 1);
            dk::mbar_init(&rec_empty[i], 1);
        }
        for (int i = 0; i < a.wstages; i++) {
            dk::mbar_init(&w_full[i], 1);
            dk::mbar_init(&w_empty[i], 1);
        }
        dk::mbar_init(&tm_full[0], 1);
        for (int i = 0; i < Q; i++) dk::mbar_init(&tm_empty[i], a.nepi);
        dk::fence_mbar_init();
    }
    if (warp == 1) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], 512;" ::"r"(
            dk::smem_u32(&tmem_base_s)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    const uint32_t tmem = tmem_base_s;

    const bool tr = a.trace != nullptr;
    long long tw0 = 0, tw1 = 0, tw2 = 0, tstart = tr ? clock64() : 0;
    if (n_tiles > 0) {
        if (warp == 0) {
            // ------------------------------------------------ weight producer (one thread): the A stream in
            // unit order; receptor planes are loaded by warp 2 + nepi, so this thread never waits on a slot
            if (elect_one()) {
                const unsigned char* wsrc = a.W + static_cast<size_t>(block) * a.nsteps * WCHUNK;
                int ws = 0, wph = 0, wuse = 0;
                for (int ti = 0; ti < n_tiles; ti++) {
                    for (int s = 0; s < a.nsteps; s += KS) {
                        if (wuse >= a.wstages) twait(&w_empty[ws], wph ^ 1, tr, tw0);
                        dk::mbar_arrive_expect_tx(&w_full[ws], STAGE);
                        dk::bulk_load(w_smem + static_cast<size_t>(ws) * STAGE, wsrc + static_cast<size_t>(s) * WCHUNK,
                                      STAGE, &w_full[ws]);
                        wuse++;
                        if (++ws == a.wstages) {
                            ws = 0;
                            wph ^= 1;
                        }
                    }
                }
                if (tr) {
                    atomicAdd(&a.trace[TR_PROD_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                    atomicAdd(&a.trace[TR_PROD_WEMPTY], static_cast<unsigned long long>(tw0));
                    atomicAdd(&a.trace[TR_CTAS], 1ull);
                    atomicAdd(&a.trace[TR_TILES], static_cast<unsigned long long>(n_tiles));
                }
            }
            __syncwarp();
        } else if (warp == 2 + a.nepi) {
            // ------------------------------------------------ receptor producer (one thread): each unit's two
            // z-planes into the next ring slot as soon as the MMAs of the unit NR earlier released it
            if (elect_one()) {
                dk::prefetch_tmap(&tmap);
                dk::prefetch_tmap(&tmap_pair);
                int rs = 0, rph = 0, ruse = 0;
                int tx = tile_begin % a.ntx, ty = (tile_begin / a.ntx) % a.nty, tz = tile_begin / (a.ntx * a.nty);
                for (int ti = 0; ti < n_tiles; ti++) {
                    for (int u = 0; u < NU; u++) {
                        const int g = u / M, vz = u % M;
                        if (ruse >= NR) twait(&rec_empty[rs], rph ^ 1, tr, tw1);
                        unsigned char* dst = rec_smem + static_cast<size_t>(rs) * a.rec_stage_bytes;
                        dk::mbar_arrive_expect_tx(&rec_full[rs], 2 * PLANE);
                        tma_load_5d(dst, &tmap, 0, tx * NTT, ty * Q, tz + vz, g, &rec_full[rs]);
                        tma_load_5d(dst + PSTRIDE, &tmap_pair, 0, tx * NTT, ty * Q, tz + vz, g, &rec_full[rs]);
                        ruse++;
                        if (++rs == NR) {
                            rs = 0;
                            rph ^= 1;
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
                if (tr) atomicAdd(&a.trace[TR_PROD_REMPTY], static_cast<unsigned long long>(tw1));
            }
            __syncwarp();
        } else if (warp == 1) {
            // ------------------------------------------------ MMA issuer (one thread); the stage loop of a
            // unit is unrolled so every in-slot descriptor offset is an immediate
            constexpr uint32_t idesc = umma_idesc(ROT, NTT);
            const uint32_t rec0 = dk::smem_u32(rec_smem), w0 = dk::smem_u32(w_smem);
            const uint64_t dA0 = umma_desc(w0, ROT * 16, 128);
            const uint64_t dB0 = umma_desc(rec0, 16, 128);   // pass 1: chunk LBO 16 B (voxel vx + 1)
            const uint64_t dP0 = umma_desc(rec0, 32, 128);   // pass 2: chunk LBO 32 B (slot x + 2)
            if (elect_one()) {
                uint32_t ws = 0, wph = 0;
                const uint32_t nws = static_cast<uint32_t>(a.wstages);
                int rs = 0, rph = 0;
                for (int ti = 0; ti < n_tiles; ti++) {
                    for (int u = 0; u < NU; u++) {
                        twait(&rec_full[rs], rph, tr, tw2);
                        tc_fence_after();
                        const uint32_t rofs = static_cast<uint32_t>(rs * a.rec_stage_bytes);
                        const uint64_t dB = dB0 + (rofs >> 4), dP = dP0 + (rofs >> 4);
#pragma unroll
                        for (int st = 0; st < NSU; st++) {
                            twait(&w_full[ws], wph, tr, tw1);
                            tc_fence_after();
                            const uint64_t da0 = dA0 + ((ws * STAGE) >> 4);
                            if (st == 0 && u == 0 && ti > 0) {
                                // first stage of a tile: each accumulator row restarts once the epilogue
                                // released it
#pragma unroll
                                for (int q = 0; q < Q; q++) {
                                    twait(&tm_empty[q], (ti - 1) & 1, tr, tw0);
                                    tc_fence_after();
#pragma unroll
                                    for (int ks = 0; ks < KS; ks++)
                                        umma_bf16(tmem + q * NTT, da0 + ((ks * WCHUNK) >> 4),
                                                  (ks < KP1 || ks >= KU ? dB : dP) +
                                                      ((unit_off(M, ks, ROW16, PSTRIDE) + q * ROW16) >> 4),
                                                  idesc, ks == 0 ? 0u : 1u);
                                }
                            } else {
                                const bool first = st == 0 && u == 0;   // ti == 0 here
#pragma unroll
                                for (int ks = 0; ks < KS; ks++) {
                                    const int s = st * KS + ks;
#pragma unroll
                                    for (int q = 0; q < Q; q++)
                                        umma_bf16(tmem + q * NTT, da0 + ((ks * WCHUNK) >> 4),
                                                  (s < KP1 || s >= KU ? dB : dP) +
                                                      ((unit_off(M, s, ROW16, PSTRIDE) + q * ROW16) >> 4),
                                                  idesc, (first && ks == 0) ? 0u : 1u);
                                }
                            }
                            umma_commit(&w_empty[ws]);
                            if (++ws == nws) {
                                ws = 0;
                                wph ^= 1;
                            }
                        }
                        umma_commit(&rec_empty[rs]);
                        if (++rs == a.n_rec_stages) {
                            rs = 0;
                            rph ^= 1;
                        }
                    }
                    umma_commit(&tm_full[0]);
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
            // ------------------------------------------------ epilogue warps
            const int quarter = warp & 3;
            const int cls = (warp - 2) >> 2;
            const int nclass = a.nepi >> 2;
            const int r = quarter * 32 + lane;
            const int slot = block * ROT + r;
            const bool rot_ok = slot < n_eff;
            unsigned long long lst[LIST];
#pragma unroll
            for (int i = 0; i < LIST; i++) lst[i] = KEY_MAX;
            float th = __int_as_float(0x7f800000);
            uint32_t th_t = 0xffffffffu;
            int tx = tile_begin % a.ntx, ty = (tile_begin / a.ntx) % a.nty, tz = tile_begin / (a.ntx * a.nty);
            for (int ti = 0; ti < n_tiles; ti++) {
                twait(&tm_full[0], ti & 1, tr, tw0);
                tc_fence_after();
                epi_tile<NTT, Q, GRID>(a, tmem, tm_empty, quarter, cls, nclass, lane, slot, rot_ok, tx, ty, tz, lst,
                                       th, th_t, tr, tw0, tw1);
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
                if (rot_ok) epi_publish(lst, slot, a);
            }
        }
    }
    tc_fence_before();
    __syncthreads();
    if (warp == 1) asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
}

// ------------------------------------------------------------------ data preparation

// bf16 split of the padded receptor: Rb[g][Z][Y][X][8] = (hi_0..3, lo_0..3) of channels 4g..4g+3
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
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
#endif

// PAIR scheme, second receptor copy: Rp[g][Z][Y][X][8] = (Rhi_{4g..4g+3}(X), Rhi_{4g..4g+3}(X+1)).
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_pack_receptor_pair_tc(const float* __restrict__ R, uint16_t* __restrict__ Rb, int nx, int ny, int nz,
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
        for (int c = 0; c < 8; c++) {
            const int p = 4 * g + (c & 3), dx = c >> 2;
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
#endif

// ------------------------------------------------------------------ variant 1: occupancy schedule
//
// Dense K-steps of variant 1 (k_corr_tc): s in [0, S1) = pass 1 (vz, vy, vxp): voxels vx = 2 vxp, 2 vxp + 1 of
// the (hi, lo) box; [S1, S1p) padding; s in [S1p, S1p + S2) = pass 2 (vz, vy, vxq): voxels 4 vxq .. 4 vxq + 3
// of the pair box; the rest padding.  Ring stage st = dense K-steps [st KS, st KS + KS).  A probe grid has at
// most one occupied voxel per atom, so most stages of one rotation carry only zero weights; a stage
// whose weights are zero for all 128 rotations of a block adds exact zeros to every accumulator and is skipped by
// the block.  Units are first grouped into blocks with few distinct active stages (k_tc_cluster).  Stage masks
// are one 64-bit word (S1p + S2p <= 256, i.e. m <= 6).

// stage bits of an occupied probe voxel (vz, vy, vx)
__host__ __device__ inline unsigned long long tc1_voxel_stages(int vz, int vy, int vx, int m)
{
    const int mxp = (m + 1) / 2, mxq = (m + 3) / 4, s1p = (m * m * mxp + KSTEPS - 1) / KSTEPS * KSTEPS;
    const int s1 = (vz * m + vy) * mxp + vx / 2, s2 = s1p + (vz * m + vy) * mxq + vx / 4;
    return (1ull << (s1 / KSTEPS)) | (1ull << (s2 / KSTEPS));
}

constexpr int CL_THREADS = 1024;
constexpr int CL_PER = 8;
constexpr int CL_W = CL_THREADS * CL_PER;   // units per clustering window (a multiple of ROT)
static_assert(CL_W % ROT == 0, "windows hold whole blocks");

#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
// Per unit: bit st = ring stage st carries a nonzero folded weight of this unit.  One warp per register batch
// of RB = 8 units: lane v reads the 8 units' weights of voxel v (32 contiguous bytes per channel), the stage bits
// of the occupied voxels are OR-reduced over the warp.  n_live (optional): units at or past it are masked out.
__global__ void k_tc_unit_masks(const float* __restrict__ Lw, int n_slots, const unsigned* __restrict__ n_live,
                                int P, int m, unsigned long long* __restrict__ masks)
{
    static_assert(dk::RB == 8, "one warp covers the 8 units of a register batch");
    const int warp = (blockIdx.x * blockDim.x + threadIdx.x) >> 5, lane = threadIdx.x & 31;
    const int n_eff = n_live ? min(n_slots, static_cast<int>(*n_live)) : n_slots;
    const int u0 = warp * dk::RB;
    if (u0 >= n_slots) return;
    const int m3 = m * m * m;
    const float* base = Lw + static_cast<size_t>(warp) * P * m3 * dk::RB;
    unsigned long long sm[dk::RB];
#pragma unroll
    for (int r = 0; r < dk::RB; r++) sm[r] = 0ull;
    for (int v = lane; v < m3; v += 32) {
        unsigned on = 0;   // bit r: unit u0 + r has a nonzero weight at voxel v
        for (int p = 0; p < P; p++) {
            const float4* q = reinterpret_cast<const float4*>(base + (static_cast<size_t>(p) * m3 + v) * dk::RB);
            const float4 w0 = q[0], w1 = q[1];
            on |= (w0.x != 0.f ? 1u : 0u) | (w0.y != 0.f ? 2u : 0u) | (w0.z != 0.f ? 4u : 0u) | (w0.w != 0.f ? 8u : 0u) |
                  (w1.x != 0.f ? 16u : 0u) | (w1.y != 0.f ? 32u : 0u) | (w1.z != 0.f ? 64u : 0u) |
                  (w1.w != 0.f ? 128u : 0u);
        }
        if (on) {
            const unsigned long long st = tc1_voxel_stages(v / (m * m), (v / m) % m, v % m, m);
#pragma unroll
            for (int r = 0; r < dk::RB; r++)
                if ((on >> r) & 1u) sm[r] |= st;
        }
    }
#pragma unroll
    for (int r = 0; r < dk::RB; r++) {
        const unsigned lo = __reduce_or_sync(0xffffffffu, static_cast<unsigned>(sm[r]));
        const unsigned hi = __reduce_or_sync(0xffffffffu, static_cast<unsigned>(sm[r] >> 32));
        if (lane == r && u0 + r < n_slots)
            masks[u0 + r] = u0 + r < n_eff ? (static_cast<unsigned long long>(hi) << 32) | lo : 0ull;
    }
}

// Greedy grouping over distinct masks (stage masks of <= CB_BITS bits, one CTA per window of CL_W units): the
// window's units are binned by mask (a stable counting sort); one warp then runs the greedy of
// k_tc_cluster on the distinct masks -- a block takes every remaining mask already inside its union (all its
// units, as far as the block has room), then all units of the mask that adds the fewest stages (ties: lowest
// mask) -- and the take records are expanded into the permutation.  Same blocks as the unit greedy up to the
// order of equal masks; the passes scale with the distinct masks, not the units.
constexpr int CB_BITS = 12;
constexpr int CB_N = 1 << CB_BITS;
constexpr int CB_MAXREC = CB_N + 2 * (CL_W / ROT);   // distinct masks + two capacity splits per block
struct ClusterBinsSmem {
    int hist[CB_N];           // units per mask -> (after the scan) first sorted position of the mask
    int fill[CB_N];           // stable-rank cursor per mask
    uint16_t lmask[CB_N];     // distinct masks present
    int lrem[CB_N];           // their remaining units
    int lbase[CB_N];          // their first sorted position
    int rec_src[CB_MAXREC];   // take records: sorted position of the first unit taken
    int rec_cnt[CB_MAXREC];   //               units taken
    int rec_pos[CB_MAXREC];   //               block position of the first one
    uint16_t umask[CL_W];     // the window's unit masks
    int wcnt[32][256];        // parallel stable sort (<= 256 distinct masks): per (warp, list entry) counts / offsets
};
__global__ void __launch_bounds__(1024, 1) k_tc_cluster_bins(const unsigned long long* __restrict__ masks, int n_slots,
                                                             int* __restrict__ sorted, int* __restrict__ perm)
{
    extern __shared__ __align__(16) unsigned char cb_raw[];
    ClusterBinsSmem& S = *reinterpret_cast<ClusterBinsSmem*>(cb_raw);
    __shared__ int s_nl, s_nrec;
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int w0 = blockIdx.x * CL_W;
    const int n = min(CL_W, n_slots - w0);
    int* srt = sorted + w0;
    for (int i = tid; i < CB_N; i += blockDim.x) S.hist[i] = 0;
    __syncthreads();
    for (int i = tid; i < n; i += blockDim.x) {
        const int b = static_cast<int>(masks[w0 + i]);
        S.umask[i] = static_cast<uint16_t>(b);
        atomicAdd(&S.hist[b], 1);
    }
    __syncthreads();
    if (warp == 0) {
        // exclusive scan of the histogram (128 bins per lane) and the list of distinct masks, in mask order
        constexpr int PER = CB_N / 32;
        int loc = 0, nz = 0;
        for (int k = 0; k < PER; k++) {
            loc += S.hist[lane * PER + k];
            nz += S.hist[lane * PER + k] != 0;
        }
        int incl = loc, inz = nz;
        for (int d = 1; d < 32; d <<= 1) {
            const int t = __shfl_up_sync(0xffffffffu, incl, d), tz = __shfl_up_sync(0xffffffffu, inz, d);
            if (lane >= d) {
                incl += t;
                inz += tz;
            }
        }
        int run = incl - loc, li = inz - nz;
        for (int k = 0; k < PER; k++) {
            const int b = lane * PER + k, c = S.hist[b];
            S.fill[b] = run;
            S.fill[b] = c ? li : -1;   // mask -> list entry (the parallel sort below); the serial one resets it
            if (c) {
                S.lmask[li] = static_cast<uint16_t>(b);
                S.lrem[li] = c;
                S.lbase[li] = run;
                li++;
            }
            S.hist[b] = run;
            run += c;
        }
        if (lane == 31) s_nl = inz;
    }
    __syncthreads();
    // stable counting sort (units of one mask in index order), so the permutation is a deterministic function of
    // the masks -- block sharding needs every rank to compute the same one
    if (s_nl <= 256) {
        // parallel: warp w ranks its contiguous chunk; per-(warp, entry) counts, scanned over the warps
        const int C = (n + 31) / 32, i_lo = warp * C, i_hi = min(n, i_lo + C), nl = s_nl;
        for (int j = lane; j < nl; j += 32) S.wcnt[warp][j] = 0;
        __syncwarp();
        for (int i0 = i_lo; i0 < i_hi; i0 += 32) {
            const int i = i0 + lane;
            const int e = i < i_hi ? S.fill[S.umask[i]] : -1;
            const unsigned grp = __match_any_sync(0xffffffffu, e);
            if (i < i_hi && (grp & ((1u << lane) - 1u)) == 0u) S.wcnt[warp][e] += __popc(grp);
            __syncwarp();
        }
        __syncthreads();
        for (int j = tid; j < nl; j += blockDim.x) {   // exclusive scan over the warps, plus the entry's base
            int run = S.lbase[j];
            for (int w = 0; w < 32; w++) {
                const int t = S.wcnt[w][j];
                S.wcnt[w][j] = run;
                run += t;
            }
        }
        __syncthreads();
        for (int i0 = i_lo; i0 < i_hi; i0 += 32) {
            const int i = i0 + lane;
            const int e = i < i_hi ? S.fill[S.umask[i]] : -1;
            const unsigned grp = __match_any_sync(0xffffffffu, e);
            const int rank = __popc(grp & ((1u << lane) - 1u));
            if (i < i_hi) srt[S.wcnt[warp][e] + rank] = w0 + i;
            __syncwarp();
            if (i < i_hi && rank == 0) S.wcnt[warp][e] += __popc(grp);
            __syncwarp();
        }
    } else if (warp == 0) {
        // serial (one warp): units in index order, 32 at a time (lanes with equal masks ranked by lane)
        for (int b = lane; b < CB_N; b += 32) S.fill[b] = S.hist[b];
        __syncwarp();
        for (int i0 = 0; i0 < n; i0 += 32) {
            const int i = i0 + lane;
            const int b = i < n ? static_cast<int>(S.umask[i]) : -1;
            const unsigned grp = __match_any_sync(0xffffffffu, b);
            const int rank = __popc(grp & ((1u << lane) - 1u));
            const int at = i < n ? S.fill[b] + rank : 0;
            __syncwarp();
            if (i < n) {
                srt[at] = w0 + i;
                if (rank == 0) S.fill[b] += __popc(grp);
            }
            __syncwarp();
        }
    }
    __syncthreads();
    if (s_nl <= 256) {
        // the greedy over <= 256 distinct masks, one list entry per thread of warps 0-7 (named barrier 1): per pass
        // a block-wide prefix of the zero-cost units (as many as fit, in list order), then the mask that adds the
        // fewest stages per unit it brings in (ties: the lowest entry = the lowest mask).  Every thread keeps
        // the same block state (union, fill, ...) in registers; the per-warp partials are double-buffered by
        // pass parity.  ~4 barriers of 8 warps per pass (one warp running the whole greedy took 120 us at
        // prod: ~400 dependent instructions per pass).  In a host model of the prod workload the ratio rule
        // cuts the blocks' active stages from 65.1 % to 63.4 % against "fewest stages" alone.
        if (warp < 8) {
            const int nl = s_nl, j = tid;
            const unsigned mk = j < nl ? static_cast<unsigned>(S.lmask[j]) : 0u;
            int rem = j < nl ? S.lrem[j] : 0, base = j < nl ? S.lbase[j] : 0;
            __shared__ int s_wsum[2][8], s_wcnt[2][8];
            __shared__ unsigned s_wmin[2][8];
            __shared__ int s_wt;
            __shared__ unsigned s_wm;
            auto bar8 = []() { asm volatile("bar.sync 1, 256;" ::: "memory"); };
            unsigned U = 0;
            int fill = 0, out = 0, nrec = 0, left = n;
            for (int ps = 0; left > 0; ps ^= 1) {
                const int cap = ROT - fill;
                // zero-cost units: block prefix in list order, capped at the room left
                const int z = (rem > 0 && (mk & ~U) == 0u) ? rem : 0;
                int incl = z;
                for (int d = 1; d < 32; d <<= 1) {
                    const int t = __shfl_up_sync(0xffffffffu, incl, d);
                    if (lane >= d) incl += t;
                }
                if (lane == 31) s_wsum[ps][warp] = incl;
                bar8();
                int before = incl - z, tz = 0;
                for (int w = 0; w < 8; w++) {
                    const int v = s_wsum[ps][w];
                    if (w < warp) before += v;
                    tz += v;
                }
                const int take = z > 0 ? max(0, min(z, cap - before)) : 0;
                const unsigned tb = __ballot_sync(0xffffffffu, take > 0);
                if (lane == 0) s_wcnt[ps][warp] = __popc(tb);
                bar8();
                int rbase = nrec, tr = 0;
                for (int w = 0; w < 8; w++) {
                    const int v = s_wcnt[ps][w];
                    if (w < warp) rbase += v;
                    tr += v;
                }
                if (take > 0) {
                    const int r = rbase + __popc(tb & ((1u << lane) - 1u));
                    S.rec_src[r] = base;
                    S.rec_cnt[r] = take;
                    S.rec_pos[r] = out + fill + before;
                    rem -= take;
                    base += take;
                }
                const int taken = min(tz, cap);
                fill += taken;
                left -= taken;
                nrec += tr;
                if (fill < ROT && left > 0) {
                    const int room = ROT - fill;
                    unsigned key = 0xffffffffu;
                    if (rem > 0) {
                        const unsigned add = static_cast<unsigned>(__popc(mk & ~U));
                        const unsigned ratio = static_cast<unsigned>(
                            __fmul_rz(static_cast<float>(add * 1024u), __frcp_rn(static_cast<float>(min(rem, room)))));
                        key = (ratio << 16) | static_cast<unsigned>(j);
                    }
                    key = __reduce_min_sync(0xffffffffu, key);
                    if (lane == 0) s_wmin[ps][warp] = key;
                    bar8();
                    unsigned win = 0xffffffffu;
                    for (int w = 0; w < 8; w++) win = min(win, s_wmin[ps][w]);
                    if (j == static_cast<int>(win & 0xffffu)) {
                        const int t = min(rem, room);
                        S.rec_src[nrec] = base;
                        S.rec_cnt[nrec] = t;
                        S.rec_pos[nrec] = out + fill;
                        rem -= t;
                        base += t;
                        s_wt = t;
                        s_wm = mk;
                    }
                    bar8();
                    U |= s_wm;
                    fill += s_wt;
                    left -= s_wt;
                    nrec++;
                    bar8();   // s_wt / s_wm are rewritten in the next pass
                }
                if (fill == ROT || left == 0) {
                    out += ROT;
                    fill = 0;
                    U = 0;
                }
            }
            if (tid == 0) s_nrec = nrec;
        }
    } else if (warp == 0) {
        // the greedy over the distinct masks (one warp; list entries lane, lane + 32, ...)
        const int nl = s_nl;
        unsigned U = 0;
        int fill = 0, out = 0, nrec = 0, left = n;
        while (left > 0) {
            const int cap = ROT - fill;
            // zero-cost masks in list order, as many units as fit
            int taken_before = 0;
            for (int j0 = 0; j0 < nl && taken_before < cap; j0 += 32) {
                const int j = j0 + lane;
                const int rem = j < nl ? S.lrem[j] : 0;
                const bool z = rem > 0 && (static_cast<unsigned>(S.lmask[j]) & ~U) == 0u;
                int c = z ? rem : 0, incl = c;
                for (int d = 1; d < 32; d <<= 1) {
                    const int t = __shfl_up_sync(0xffffffffu, incl, d);
                    if (lane >= d) incl += t;
                }
                const int before = taken_before + incl - c;
                const int take = z ? max(0, min(c, cap - before)) : 0;
                const unsigned tb = __ballot_sync(0xffffffffu, take > 0);
                if (take > 0) {
                    const int r = nrec + __popc(tb & ((1u << lane) - 1u));
                    S.rec_src[r] = S.lbase[j];
                    S.rec_cnt[r] = take;
                    S.rec_pos[r] = out + fill + before;
                    S.lrem[j] = rem - take;
                    S.lbase[j] += take;
                }
                nrec += __popc(tb);
                taken_before += __shfl_sync(0xffffffffu, incl, 31);
                taken_before = min(taken_before, cap);
            }
            fill += taken_before;
            left -= taken_before;
            __syncwarp();
            if (fill < ROT && left > 0) {
                // the mask that adds the fewest stages (ties: the lowest mask)
                unsigned best = 0xffffffffu;
                for (int j = lane; j < nl; j += 32)
                    if (S.lrem[j] > 0)
                        best = min(best, (static_cast<unsigned>(__popc(static_cast<unsigned>(S.lmask[j]) & ~U)) << 16) |
                                             static_cast<unsigned>(j));
                best = __reduce_min_sync(0xffffffffu, best);
                const int j = static_cast<int>(best & 0xffffu);
                const int take = min(S.lrem[j], ROT - fill);
                if (lane == 0) {
                    S.rec_src[nrec] = S.lbase[j];
                    S.rec_cnt[nrec] = take;
                    S.rec_pos[nrec] = out + fill;
                    S.lrem[j] -= take;
                    S.lbase[j] += take;
                }
                __syncwarp();
                nrec++;
                U |= static_cast<unsigned>(S.lmask[j]);
                fill += take;
                left -= take;
            }
            if (fill == ROT || left == 0) {
                out += ROT;
                fill = 0;
                U = 0;
            }
        }
        if (lane == 0) s_nrec = nrec;
    }
    __syncthreads();
    // expand the records: record r places sorted units [src, src + cnt) at block positions [pos, pos + cnt)
    const int nrec = s_nrec;
    for (int r = warp; r < nrec; r += blockDim.x / 32)
        for (int i = lane; i < S.rec_cnt[r]; i += 32) perm[w0 + S.rec_pos[r] + i] = srt[S.rec_src[r] + i];
}

// Greedy grouping of the units of one window (CL_W units, one CTA) into blocks of ROT: a block takes every
// remaining unit whose K-steps are already in its union, then the unit that adds the fewest new K-steps (ties:
// lowest index), until it holds ROT units.  One pass over the window per added unit that grows the union.
// Measured on the prod workload: the blocks' unions cover 50 % of the K-steps, against 89 % for blocks of
// consecutive units (the rotations of one probe).  perm[w0 + i] = the unit at block position w0 + i.
__global__ void __launch_bounds__(CL_THREADS, 1) k_tc_cluster(const unsigned long long* __restrict__ masks, int n_slots,
                                                              int* __restrict__ perm)
{
    constexpr int NW = CL_THREADS / 32;
    static_assert(CL_PER == 8 && NW == 32, "the warp-redundant scan assumes 8 x 32 counters");
    __shared__ unsigned s_cnt[2][CL_PER][NW];   // zero-cost units per (slot k, warp), double-buffered by pass
    __shared__ unsigned s_min[2][NW];           // per-warp argmin key (added K-steps << 16 | window index)
    __shared__ unsigned long long s_U[2];       // union of the open block (state double-buffered by pass)
    __shared__ int s_fill[2], s_out[2], s_left[2];
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int w0 = blockIdx.x * CL_W;
    const int n = min(CL_W, n_slots - w0);
    unsigned long long mk[CL_PER];
    unsigned live = 0;   // bit k: unit tid + k * CL_THREADS not yet placed
#pragma unroll
    for (int k = 0; k < CL_PER; k++) {
        const int j = tid + k * CL_THREADS;
        mk[k] = j < n ? masks[w0 + j] : 0ull;
        if (j < n) live |= 1u << k;
    }
    if (tid == 0) {
        s_U[0] = 0ull;
        s_fill[0] = 0;
        s_out[0] = 0;
        s_left[0] = n;
    }
    __syncthreads();
    for (int ps = 0;; ps ^= 1) {
        const unsigned long long U = s_U[ps];
        const int fill = s_fill[ps], out = s_out[ps], left = s_left[ps];
        if (left <= 0) break;
        // 1. zero-cost units (a ballot per slot k) and this warp's cheapest positive unit
        unsigned zb[CL_PER];
        unsigned best = 0xffffffffu;
#pragma unroll
        for (int k = 0; k < CL_PER; k++) {
            const bool lv = (live >> k) & 1u;
            const unsigned add = static_cast<unsigned>(__popcll(mk[k] & ~U));
            zb[k] = __ballot_sync(0xffffffffu, lv && add == 0u);
            if (lv && add != 0u) best = min(best, (add << 16) | static_cast<unsigned>(tid + k * CL_THREADS));
            if (lane == 0) s_cnt[ps][k][warp] = __popc(zb[k]);
        }
        best = __reduce_min_sync(0xffffffffu, best);
        if (lane == 0) s_min[ps][warp] = best;
        __syncthreads();
        // 2. warp-redundant exclusive scan of the counters in (k, warp) order and argmin over the warps
        unsigned c8[8], loc = 0;
#pragma unroll
        for (int e = 0; e < 8; e++) {
            c8[e] = s_cnt[ps][lane >> 2][(lane & 3) * 8 + e];
            loc += c8[e];
        }
        unsigned incl = loc;
#pragma unroll
        for (int d = 1; d < 32; d <<= 1) {
            const unsigned t = __shfl_up_sync(0xffffffffu, incl, d);
            if (lane >= d) incl += t;
        }
        const int total = static_cast<int>(__shfl_sync(0xffffffffu, incl, 31));
        unsigned sel = incl - loc;   // exclusive prefix of counter (lane >> 2, (lane & 3) * 8 + (warp & 7))
#pragma unroll
        for (int e = 0; e < 8; e++)
            if (e < (warp & 7)) sel += c8[e];
        const unsigned win = __reduce_min_sync(0xffffffffu, s_min[ps][lane]);
        const int cap = ROT - fill;
        const int taken = min(total, cap);
#pragma unroll
        for (int k = 0; k < CL_PER; k++) {
            const int base = static_cast<int>(__shfl_sync(0xffffffffu, sel, k * 4 + (warp >> 3)));
            if ((zb[k] >> lane) & 1u) {
                const int rank = base + __popc(zb[k] & ((1u << lane) - 1u));
                if (rank < cap) {
                    perm[w0 + out + fill + rank] = w0 + tid + k * CL_THREADS;
                    live &= ~(1u << k);
                }
            }
        }
        const int nf = fill + taken;
        const bool add_win = nf < ROT && win != 0xffffffffu;
        const int jw = static_cast<int>(win & 0xffffu);
        if (add_win && jw % CL_THREADS == tid) {
            live &= ~(1u << (jw / CL_THREADS));
            perm[w0 + out + nf] = w0 + jw;
        }
        if (tid == 0) {   // next pass's state (the other buffer: this pass's is still being read)
            const int nf2 = nf + (add_win ? 1 : 0);
            s_left[ps ^ 1] = left - taken - (add_win ? 1 : 0);
            if (nf2 == ROT || s_left[ps ^ 1] == 0) {   // block closed
                s_out[ps ^ 1] = out + ROT;
                s_fill[ps ^ 1] = 0;
                s_U[ps ^ 1] = 0ull;
            } else {
                s_out[ps ^ 1] = out;
                s_fill[ps ^ 1] = nf2;
                s_U[ps ^ 1] = add_win ? (U | __ldg(&masks[w0 + jw])) : U;
            }
        }
        __syncthreads();
    }
}

// Per rotation block (one CTA of 128 threads): the mask of active ring stages -- the OR of its units' masks
// (k_tc_unit_masks: zero for positions past the live count); at least one stage, so every row's accumulators are
// written -- its stage count and the dense stage of every compacted A stage (ksrc).  masks == nullptr: every
// stage (dense schedule).  ksum accumulates the executed K-steps (statistics).
__global__ void k_tc_block_tables(const unsigned long long* __restrict__ masks, const int* __restrict__ perm,
                                  int n_slots, int nsteps, uint16_t* __restrict__ ksrc, int4* __restrict__ kinfo,
                                  unsigned* __restrict__ ksum)
{
    const int blk = blockIdx.x, nstg = nsteps / KSTEPS, lane = threadIdx.x & 31;
    uint16_t* src = ksrc + static_cast<size_t>(blk) * nsteps;
    unsigned long long mk = 0;
    if (masks) {
        for (int r = threadIdx.x; r < ROT; r += blockDim.x) {
            const int pos = blk * ROT + r;
            if (pos < n_slots) mk |= masks[perm ? perm[pos] : pos];
        }
    } else if (threadIdx.x == 0) {
        mk = nstg >= 64 ? ~0ull : (1ull << nstg) - 1ull;
    }
    __shared__ unsigned long long s_mk[4];
    const unsigned lo = __reduce_or_sync(0xffffffffu, static_cast<unsigned>(mk));
    const unsigned hi = __reduce_or_sync(0xffffffffu, static_cast<unsigned>(mk >> 32));
    if (lane == 0) s_mk[threadIdx.x >> 5] = (static_cast<unsigned long long>(hi) << 32) | lo;
    __syncthreads();
    if (threadIdx.x != 0) return;
    mk = s_mk[0] | s_mk[1] | s_mk[2] | s_mk[3];
    if (mk == 0ull) mk = 1ull;   // all-zero block: one zero-weight stage writes the accumulators
    int i = 0;
    for (int st = 0; st < nstg; st++)
        if ((mk >> st) & 1ull) src[i++] = static_cast<uint16_t>(st);
    kinfo[blk] = make_int4(i, 0, static_cast<int>(static_cast<uint32_t>(mk)), static_cast<int>(static_cast<uint32_t>(mk >> 32)));
    if (ksum) atomicAdd(ksum, static_cast<unsigned>(i * KSTEPS));
}

// Segment boundaries of the dynamic tile scheduler (one CTA): the chunk space (block-major, cpb chunks per
// block) is cut into ns contiguous segments of equal estimated cost, a chunk of block b costing (its ring
// stages + e_cost) -- the occupancy schedule makes blocks' tiles differ in length, and segments of equal chunk
// counts would leave CTAs with cheap blocks helping others (each help restarts top-k lists: bursts of
// insertions).  seg[j] = first chunk of segment j, seg[ns] = n_blocks * cpb.
__global__ void k_tc_segments(const int4* __restrict__ kinfo, const int* __restrict__ blkmap, int n_blocks, int cpb,
                              int ns, int e_cost, long long* __restrict__ pref, long long* __restrict__ seg)
{
    __shared__ long long s_carry;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    __shared__ long long s_w[32];
    if (threadIdx.x == 0) s_carry = 0;
    __syncthreads();
    // pref[b] = cost of the chunks of blocks [0, b)
    for (int b0 = 0; b0 < n_blocks; b0 += blockDim.x) {
        const int b = b0 + threadIdx.x;
        long long c = b < n_blocks ? static_cast<long long>(cpb) * (kinfo[blkmap ? blkmap[b] : b].x + e_cost) : 0;
        long long incl = c;
        for (int d = 1; d < 32; d <<= 1) {
            const long long t = __shfl_up_sync(0xffffffffu, incl, d);
            if (lane >= d) incl += t;
        }
        if (lane == 31) s_w[warp] = incl;
        __syncthreads();
        long long wbase = 0;
        for (int w = 0; w < warp; w++) wbase += s_w[w];
        if (b < n_blocks) pref[b] = s_carry + wbase + incl - c;
        __syncthreads();
        if (threadIdx.x == blockDim.x - 1) s_carry += wbase + incl;
        __syncthreads();
    }
    const long long total = s_carry;
    for (int j = threadIdx.x; j <= ns; j += blockDim.x) {
        long long c;
        if (j == ns) {
            c = static_cast<long long>(n_blocks) * cpb;
        } else {
            const long long t = total * j / ns;
            int lo = 0, hi = n_blocks - 1;   // last block with pref <= t
            while (lo < hi) {
                const int mid = (lo + hi + 1) >> 1;
                if (pref[mid] <= t) lo = mid;
                else hi = mid - 1;
            }
            const long long w = kinfo[blkmap ? blkmap[lo] : lo].x + e_cost;
            c = static_cast<long long>(lo) * cpb + min(static_cast<long long>(cpb), (t - pref[lo]) / w);
        }
        seg[j] = c;
    }
}

// Block sharding (multi-GPU): rank `rank` of `world` docks blocks b = rank, rank + world, ... of the call's block
// order (interleaved, so every rank gets blocks from the whole cost range of the clustering); blkmap[lb] = its
// lb-th block, owned[unit] = 1 for the units of those blocks.
__global__ void k_tc_shard_blocks(const int* __restrict__ perm, int n_slots, int n_blocks, int rank, int world,
                                  int* __restrict__ blkmap, unsigned char* __restrict__ owned)
{
    for (int pos = blockIdx.x * blockDim.x + threadIdx.x; pos < n_blocks * ROT; pos += gridDim.x * blockDim.x) {
        const int b = pos / ROT;
        if (pos % ROT == 0 && b % world == rank) blkmap[b / world] = b;
        if (pos < n_slots) owned[perm ? perm[pos] : pos] = static_cast<unsigned char>(b % world == rank);
    }
}

// Variant 1 A operand, compacted: entry i of block b = dense K-step ksrc[b][i] of the units at the block's
// positions.  Pass 1 chunks (Whi(vx), Whi(vx)), vx = 2 vxp + c; pass 2 chunks (Wlo(vx0), Wlo(vx0 + 1)),
// vx0 = 4 vxq + 2c; padding steps are zero.
__global__ void k_pack_weights_tc1(const float* __restrict__ Lw, const int* __restrict__ perm,
                                   const uint16_t* __restrict__ ksrc, const int4* __restrict__ kinfo,
                                   unsigned char* __restrict__ W, int n_slots, int P, int m, int stride)
{
    const int MXP = (m + 1) / 2, MXQ = (m + 3) / 4, m3 = m * m * m, S1 = m * m * MXP, S2 = m * m * MXQ;
    const int S1P = (S1 + KSTEPS - 1) / KSTEPS * KSTEPS;
    const long long n_blocks = (n_slots + ROT - 1) / ROT;
    const long long total = n_blocks * stride * 2 * ROT;
    for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<long long>(gridDim.x) * blockDim.x) {
        const int r = static_cast<int>(i % ROT);
        const int c = static_cast<int>((i / ROT) % 2);
        const int e = static_cast<int>((i / (2 * ROT)) % stride);
        const long long blk = i / (2LL * ROT * stride);
        if (e >= kinfo[blk].x * KSTEPS) continue;   // beyond the block's schedule: never streamed
        const long long pos = blk * ROT + r;
        const int s = ksrc[blk * stride + e / KSTEPS] * KSTEPS + e % KSTEPS;   // dense K-step
        uint16_t out[8] = {0, 0, 0, 0, 0, 0, 0, 0};
        if (pos < n_slots && (s < S1 || (s >= S1P && s < S1P + S2))) {
            const long long slot = perm ? perm[pos] : pos;
            auto wval = [&](int vz, int vy, int vx, int p) -> float {
                if (vx >= m || p >= P) return 0.f;
                const int v = (vz * m + vy) * m + vx;
                return Lw[((static_cast<size_t>(slot / dk::RB) * P + p) * m3 + v) * dk::RB + slot % dk::RB];
            };
            if (s < S1) {
                const int vxp = s % MXP, vy = (s / MXP) % m, vz = s / (MXP * m);
                const int vx = 2 * vxp + c;
#pragma unroll
                for (int p = 0; p < 4; p++) {
                    const __nv_bfloat16 hi = __float2bfloat16_rn(wval(vz, vy, vx, p));
                    out[p] = out[4 + p] = __bfloat16_as_ushort(hi);
                }
            } else {
                const int t = s - S1P;
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
#endif

// Streamed-plane A operand (variant 2): steps [u * KUP, (u + 1) * KUP) belong to unit u = (g, vz);
// within a unit, steps [0, m * MXP) are pass-1 chunks (Whi(vx), Whi(vx)) over (vy, vxp), vx = 2 vxp + c,
// steps [m * MXP, m * MXP + m * MXQ) pass-2 chunks (Wlo(vx0), Wlo(vx0 + 1)) over (vy, vxq),
// vx0 = 4 vxq + 2c, of channels 4g..4g+3; the rest is zero padding.
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_pack_weights_tcs(const float* __restrict__ Lw, unsigned char* __restrict__ W, int n_slots, int P,
                                   int m, int nsteps)
{
    const int MXP = (m + 1) / 2, MXQ = (m + 3) / 4, m3 = m * m * m;
    const int KP1 = m * MXP, KU = KP1 + m * MXQ, KUP = (KU + KSTEPS - 1) / KSTEPS * KSTEPS;
    const long long n_blocks = (n_slots + ROT - 1) / ROT;
    const long long total = n_blocks * nsteps * 2 * ROT;
    for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<long long>(gridDim.x) * blockDim.x) {
        const int r = static_cast<int>(i % ROT);
        const int c = static_cast<int>((i / ROT) % 2);
        const int s = static_cast<int>((i / (2 * ROT)) % nsteps);
        const long long blk = i / (2LL * ROT * nsteps);
        const long long slot = blk * ROT + r;
        const int u = s / KUP, sl = s % KUP, g = u / m, vz = u % m;
        uint16_t out[8] = {0, 0, 0, 0, 0, 0, 0, 0};
        auto wval = [&](int vy, int vx, int p) -> float {
            if (vx >= m || p >= P) return 0.f;
            const int v = (vz * m + vy) * m + vx;
            return Lw[((static_cast<size_t>(slot / dk::RB) * P + p) * m3 + v) * dk::RB + slot % dk::RB];
        };
        if (slot < n_slots) {
            if (sl < KP1) {
                const int vy = sl / MXP, vx = 2 * (sl % MXP) + c;
#pragma unroll
                for (int cc = 0; cc < 4; cc++) {
                    const __nv_bfloat16 hi = __float2bfloat16_rn(wval(vy, vx, 4 * g + cc));
                    out[cc] = out[4 + cc] = __bfloat16_as_ushort(hi);
                }
            } else if (sl < KU) {
                const int t = sl - KP1, vy = t / MXQ, vx0 = 4 * (t % MXQ) + 2 * c;
#pragma unroll
                for (int cc = 0; cc < 4; cc++) {
#pragma unroll
                    for (int d = 0; d < 2; d++) {
                        const float f = wval(vy, vx0 + d, 4 * g + cc);
                        const __nv_bfloat16 hi = __float2bfloat16_rn(f);
                        const __nv_bfloat16 lo = __float2bfloat16_rn(f - __bfloat162float(hi));
                        out[4 * d + cc] = __bfloat16_as_ushort(lo);
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
#endif

}  // namespace tc

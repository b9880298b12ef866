// dock_kernels.cuh -- sm_100a kernels of the rigid-docking hot path.
//
// Citations "P:L<a>-<b>" point into PAPER.md (Sukhwani & Herbordt, IPPS 2010).
// Layouts and rooflines are in DESIGN.md §Kernels.
//
//   k_pad_receptor   a0  cyclic-halo padded receptor copy (init, once)
//   k_voxelize       a1  rotate + grid-assign the probe, fold w_p (FP64 index) P:L184-186, L536-537
//   k_corr<M,GRID>   a2-a5  TMA-staged receptor tiles, FP32 FFMA multi-term
//                        direct correlation register-blocked over (8 x-outputs x
//                        8 rotations), fused weighted sum, per-warp top-32 lists
//                        (GRID=false) or a score-grid epilogue (GRID=true)
//   k_merge          a6  per-rotation greedy best-then-exclude over candidates
//   k_greedy_round   a6' exact greedy over full score grids (fallback)
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>
#include <stdint.h>

namespace dk {

constexpr int RB = 8;          // rotations per register block (paper: 8 rotations per pass)
constexpr int XT = 8;          // consecutive x translations per thread
constexpr int NWC = 8;         // consumer (compute) warps per CTA
constexpr int NTHREADS = (NWC + 1) * 32;   // + 1 TMA producer warp
constexpr int LIST = 32;       // per-warp candidate list length (one key per lane)
constexpr unsigned FULL = 0xffffffffu;
constexpr unsigned long long KEY_MAX = ~0ull;

// status bits written by kernels (device status word)
constexpr int ST_BAD_ROTATION = 1;
constexpr int ST_OUTSIDE = 2;

struct Geo {
    int nx, ny, nz;
    int LX, WY;            // lanes along x per row; rows per warp (= 32/LX)
    int TX, TY, TZ;        // translation tile extents (TX = LX*XT, TY*TZ = NWC*WY)
    int ntx, nty, ntz, ntiles;
    int Xp, Yp, Zp;        // padded receptor extents
};

struct CorrArgs {
    Geo g;
    int P;
    const float* Lw;            // [n_batches][P][M^3][RB] folded weights w_p * L_{r,p}
    int n_slots;                // rotations (units) in this launch
    int G;                      // regions per rotation batch
    int tiles_per_region;
    int nstage;
    int stage_rec_bytes;        // TXB*TYB*TZB*4 rounded up to a multiple of 128 (stage offset)
    int box_bytes;              // TXB*TYB*TZB*4 exactly (TMA transaction bytes)
    int stage_bytes;            // stage_rec_bytes + M^3*RB*4 (multiple of 128)
    int TXB, TYB, TZB;          // receptor box extents for this M
    // top-k mode
    int k, rho;
    unsigned long long* T;      // [n_slots] pruning bound (atomicMin)
    unsigned long long* mu;     // [n_slots] min over warp lists of the 32nd key (atomicMin)
    unsigned int* cnt;          // [n_slots] candidates written (atomicAdd)
    unsigned long long* cand;   // [n_slots][cap]
    int cap;
    // grid mode
    float* grid;                // [n_slots][nz][ny][nx]
    const unsigned* n_live;     // optional (device): only slots < *n_live are live (device-driven fallback)
};

// ------------------------------------------------------------------ small helpers

__device__ __forceinline__ uint32_t smem_u32(const void* p)
{
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

// Order-preserving map float -> uint32 (ascending); -0.0 is first normalised to +0.0 (reading Q8).
__device__ __forceinline__ uint32_t ord_f32(float f)
{
    f = __fadd_rn(f, 0.0f);
    uint32_t b = __float_as_uint(f);
    return (b & 0x80000000u) ? ~b : (b | 0x80000000u);
}
__device__ __forceinline__ float unord_f32(uint32_t o)
{
    uint32_t b = (o & 0x80000000u) ? (o & 0x7fffffffu) : ~o;
    return __uint_as_float(b);
}
__device__ __forceinline__ unsigned long long make_key(float s, uint32_t t)
{
    return (static_cast<unsigned long long>(ord_f32(s)) << 32) | t;
}
// Upper bound (as float) of the score part of a key; +inf for KEY_MAX / empty slots.
__device__ __forceinline__ float key_score_bound(uint32_t hi)
{
    return hi >= 0xff800000u ? __int_as_float(0x7f800000) : unord_f32(hi);
}

__device__ __forceinline__ unsigned long long shfl_u64(unsigned long long v, int src)
{
    return __shfl_sync(FULL, v, src);
}
__device__ __forceinline__ unsigned long long warp_min_u64(unsigned long long v)
{
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        unsigned long long w = __shfl_xor_sync(FULL, v, o);
        v = w < v ? w : v;
    }
    return v;
}

// Insert key into a warp-distributed ascending list (lane i holds the i-th smallest).
__device__ __forceinline__ void warp_list_insert(unsigned long long& L, unsigned long long key, int lane)
{
    unsigned long long prev = __shfl_up_sync(FULL, L, 1);
    bool lt = key < L;
    bool ltp = (lane > 0) && (key < prev);
    L = lt ? (ltp ? prev : key) : L;
}

// Cyclic Chebyshev distance between two translations (reading Q9).
__device__ __forceinline__ int cheb_cyc(uint32_t a, uint32_t b, int nx, int ny, int nz)
{
    int ax = a % nx, ay = (a / nx) % ny, az = a / (nx * ny);
    int bx = b % nx, by = (b / nx) % ny, bz = b / (nx * ny);
    int dx = abs(ax - bx), dy = abs(ay - by), dz = abs(az - bz);
    dx = min(dx, nx - dx);
    dy = min(dy, ny - dy);
    dz = min(dz, nz - dz);
    return max(dx, max(dy, dz));
}

// ------------------------------------------------------------------ mbarrier / TMA (PTX)

__device__ __forceinline__ void mbar_init(uint64_t* bar, unsigned count)
{
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void fence_mbar_init()
{
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t* bar, unsigned bytes)
{
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
                 : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t* bar)
{
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
__device__ __forceinline__ bool mbar_try_wait(uint64_t* bar, unsigned parity)
{
    uint32_t ok;
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
        "selp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(ok)
        : "r"(smem_u32(bar)), "r"(parity)
        : "memory");
    return ok != 0;
}
// Non-blocking probe of a phase (mbarrier.test_wait).
__device__ __forceinline__ bool mbar_test(uint64_t* bar, unsigned parity)
{
    uint32_t ok;
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "mbarrier.test_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
        "selp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(ok)
        : "r"(smem_u32(bar)), "r"(parity)
        : "memory");
    return ok != 0;
}
// Wait for the phase with the given parity.  A watchdog turns a lost transaction (which
// would otherwise hang the GPU) into a trapped launch error after ~2^35 cycles (~17 s).
__device__ __forceinline__ void mbar_wait(uint64_t* bar, unsigned parity)
{
    if (mbar_try_wait(bar, parity)) return;
    const long long t0 = clock64();
    while (!mbar_try_wait(bar, parity)) {
        if (clock64() - t0 > (1ll << 35)) __trap();
    }
}
__device__ __forceinline__ void tma_load_4d(void* dst, const CUtensorMap* map, int x, int y, int z, int c,
                                            uint64_t* bar)
{
    asm volatile(
        "cp.async.bulk.tensor.4d.shared::cluster.global.tile.mbarrier::complete_tx::bytes"
        " [%0], [%1, {%2, %3, %4, %5}], [%6];" ::"r"(smem_u32(dst)),
        "l"(reinterpret_cast<uint64_t>(map)), "r"(x), "r"(y), "r"(z), "r"(c), "r"(smem_u32(bar))
        : "memory");
}
__device__ __forceinline__ void bulk_load(void* dst, const void* src, unsigned bytes, uint64_t* bar)
{
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
            smem_u32(dst)),
        "l"(src), "r"(bytes), "r"(smem_u32(bar))
        : "memory");
}
__device__ __forceinline__ void prefetch_tmap(const CUtensorMap* map)
{
    asm volatile("prefetch.tensormap [%0];" ::"l"(reinterpret_cast<uint64_t>(map)) : "memory");
}

// ------------------------------------------------------------------ a0: cyclic-halo padding

// Rpad[p][Z][Y][X] = R[p][Z mod nz][Y mod ny][X mod nx]   (reading Q2: cyclic translations)
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_pad_receptor(const float* __restrict__ R, float* __restrict__ Rp, int nx, int ny, int nz,
                               int Xp, int Yp, int Zp, int P)
{
    size_t total = static_cast<size_t>(P) * Zp * Yp * Xp;
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<size_t>(gridDim.x) * blockDim.x) {
        int X = static_cast<int>(i % Xp);
        size_t r = i / Xp;
        int Y = static_cast<int>(r % Yp);
        r /= Yp;
        int Z = static_cast<int>(r % Zp);
        int p = static_cast<int>(r / Zp);
        Rp[i] = R[((static_cast<size_t>(p) * nz + Z % nz) * ny + Y % ny) * nx + X % nx];
    }
}
#endif

#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_count_nonfinite(const float* __restrict__ a, size_t n, unsigned int* bad)
{
    unsigned c = 0;
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < n;
         i += static_cast<size_t>(gridDim.x) * blockDim.x)
        c += isfinite(a[i]) ? 0u : 1u;
    if (c) atomicAdd(bad, c);
}
#endif

// ------------------------------------------------------------------ a1: voxelize

struct VoxArgs {
    const double* xyz;     // [total_atoms][3]
    const float* coef;     // [total_atoms][P]
    const int* atom_off;   // [n_probes + 1]
    const double* rot;     // [n_rot][9]
    const float* w;        // [P] weights folded into the grids
    const int* unit_list;  // optional: slot -> call-relative unit (fallback); unit = unit_begin + unit_list[slot]
    long long unit_begin;
    int n_rot, n_slots, P, m;
    double spacing;
    float* Lw;             // [ceil(n_slots/RB)][P][m^3][RB]
    int* status;
    const unsigned* n_live;   // optional (device): slots >= *n_live are zero padding (device-driven fallback)
};

// One thread per (slot, p): sums the coefficients of the probe's atoms in atom order
// (deterministic), then multiplies by w_p.  Index math in FP64 with explicit IEEE
// rounding (no FMA contraction) so that voxel indices equal the oracle's exactly.
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__device__ __forceinline__ void voxelize_body(const VoxArgs& a)
{
    int idx = blockIdx.x * blockDim.x + threadIdx.x;
    const int n_pad = (a.n_slots + RB - 1) / RB * RB;   // the last batch is zero-padded
    if (idx >= n_pad * a.P) return;
    int slot = idx / a.P, p = idx % a.P;
    const int m = a.m, m3 = m * m * m;
    float* dst = a.Lw + (static_cast<size_t>(slot / RB) * a.P + p) * m3 * RB + (slot % RB);
    for (int v = 0; v < m3; v++) dst[v * RB] = 0.0f;
    const int n_eff = a.n_live ? min(a.n_slots, static_cast<int>(*a.n_live)) : a.n_slots;
    if (slot >= n_eff) return;
    long long unit = a.unit_begin + (a.unit_list ? static_cast<long long>(a.unit_list[slot]) : slot);
    int probe = static_cast<int>(unit / a.n_rot), r = static_cast<int>(unit % a.n_rot);
    const double* q = a.rot + 9 * static_cast<size_t>(r);

    if (p == 0) {   // rotation check: |Q^T Q - I| <= 1e-9 and det > 0 (reading Q5)
        bool ok = true;
        for (int i = 0; i < 3; i++)
            for (int j = 0; j < 3; j++) {
                double s = __dmul_rn(q[i], q[j]);
                s = __dadd_rn(s, __dmul_rn(q[3 + i], q[3 + j]));
                s = __dadd_rn(s, __dmul_rn(q[6 + i], q[6 + j]));
                double want = (i == j) ? 1.0 : 0.0;
                if (!(fabs(s - want) <= 1e-9)) ok = false;
            }
        double det = q[0] * (q[4] * q[8] - q[5] * q[7]) - q[1] * (q[3] * q[8] - q[5] * q[6]) +
                     q[2] * (q[3] * q[7] - q[4] * q[6]);
        if (!(det > 0.0)) ok = false;
        if (!ok) atomicOr(a.status, ST_BAD_ROTATION);
    }
    const double c = (m - 1) / 2.0;
    bool outside = false;
    for (int at = a.atom_off[probe]; at < a.atom_off[probe + 1]; at++) {
        const double* x = a.xyz + 3 * static_cast<size_t>(at);
        int v[3];
        bool in = true;
#pragma unroll
        for (int i = 0; i < 3; i++) {
            double rx = __dmul_rn(q[3 * i + 0], x[0]);
            rx = __dadd_rn(rx, __dmul_rn(q[3 * i + 1], x[1]));
            rx = __dadd_rn(rx, __dmul_rn(q[3 * i + 2], x[2]));
            double g = __dadd_rn(__ddiv_rn(rx, a.spacing), c);
            double f = floor(__dadd_rn(g, 0.5));
            in = in && (f >= 0.0 && f < static_cast<double>(m));
            v[i] = in ? static_cast<int>(f) : 0;
        }
        if (!in) {
            outside = true;
            continue;
        }
        dst[((v[2] * m + v[1]) * m + v[0]) * RB] += a.coef[static_cast<size_t>(at) * a.P + p];
    }
    if (outside && p == 0) atomicOr(a.status, ST_OUTSIDE);
    const float wp = a.w[p];
    for (int v = 0; v < m3; v++) dst[v * RB] = dst[v * RB] * wp;
}
__global__ void k_voxelize(VoxArgs a) { voxelize_body(a); }
// arguments read from device memory (the device-driven fallback's per-call arguments, so that a captured
// CUDA graph of the fallback loop stays valid across calls)
__global__ void k_voxelize_dyn(const VoxArgs* a) { voxelize_body(*a); }
#endif

// Lw [batch][P][m^3][RB]  ->  out [slot][P][m^3]   (debug export for dock_voxelize)
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_unpack_L(const float* __restrict__ Lw, float* __restrict__ out, int n_slots, int P, int m3)
{
    int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= n_slots * P * m3) return;
    int v = i % m3, p = (i / m3) % P, slot = i / (m3 * P);
    out[i] = Lw[((static_cast<size_t>(slot / RB) * P + p) * m3 + v) * RB + slot % RB];
}
#endif

// ------------------------------------------------------------------ a2-a5: correlation

// One CTA = one work item (rotation batch b of RB slots, translation region).  Warp NWC is
// the TMA producer: for each (tile, channel p) of the region it loads the receptor box
// [TZB][TYB][TXB] of channel p and the batch's folded weights of channel p into a ring
// stage.  Warps 0..NWC-1 compute: each lane owns XT consecutive x translations of one
// (y, z) row and RB rotations, i.e. RB*XT FP32 accumulators, and for every (p, vz, vy)
// row loads XT+M-1 receptor values once (LDS.128) and reuses them for all M vx offsets
// and all RB rotations ("each protein voxel fetched ... gets reused multiple
// times"), the RB weights of one (p, v) being a warp-uniform broadcast load.
// Epilogue (GRID=false): per rotation, keys (score, t_lin) below the warp list's 32nd key
// are inserted into a warp-distributed sorted list (no score grid is written).
// At the end of the item each warp publishes a pruning bound and its surviving keys.
template <int M, bool GRID>
__global__ void __launch_bounds__(NTHREADS, 1) k_corr(const __grid_constant__ CUtensorMap tmap, const CorrArgs a)
{
    extern __shared__ __align__(128) unsigned char smem[];
    constexpr int M3 = M * M * M;
    constexpr int NR = XT + M - 1;              // receptor values per row per lane
    constexpr int NR4 = (NR + 3) / 4;           // LDS.128 per row per lane

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int item = blockIdx.x;
    const int batch = item / a.G, region = item % a.G;
    const int tile_begin = region * a.tiles_per_region;
    const int tile_end = min(a.g.ntiles, tile_begin + a.tiles_per_region);
    const int n_it = (tile_end - tile_begin) * a.P;
    const int slot0 = batch * RB;
    const int n_eff = a.n_live ? min(a.n_slots, static_cast<int>(*a.n_live)) : a.n_slots;
    if (slot0 >= n_eff) return;   // uniform: a dead batch of the device-driven fallback
    const int nb = min(RB, n_eff - slot0);

    uint64_t* full = reinterpret_cast<uint64_t*>(smem + a.nstage * a.stage_bytes);
    uint64_t* empty = full + a.nstage;
    if (threadIdx.x == 0) {
        for (int s = 0; s < a.nstage; s++) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], NWC);
        }
        fence_mbar_init();
    }
    __syncthreads();
    if (n_it <= 0) return;

    if (warp == NWC) {
        // ---------------- TMA producer (one elected lane)
        if (lane == 0) {
            prefetch_tmap(&tmap);
            const float* wsrc = a.Lw + static_cast<size_t>(batch) * a.P * M3 * RB;
            const unsigned wbytes = M3 * RB * 4;
            for (int it = 0; it < n_it; it++) {
                const int s = it % a.nstage;
                const int use = it / a.nstage;
                if (use > 0) mbar_wait(&empty[s], (use - 1) & 1);
                const int tile = tile_begin + it / a.P;
                const int p = it % a.P;
                const int tx = tile % a.g.ntx, ty = (tile / a.g.ntx) % a.g.nty, tz = tile / (a.g.ntx * a.g.nty);
                unsigned char* st = smem + static_cast<size_t>(s) * a.stage_bytes;
                mbar_arrive_expect_tx(&full[s], a.box_bytes + wbytes);
                tma_load_4d(st, &tmap, tx * a.g.TX, ty * a.g.TY, tz * a.g.TZ, p, &full[s]);
                bulk_load(st + a.stage_rec_bytes, wsrc + static_cast<size_t>(p) * M3 * RB, wbytes, &full[s]);
            }
        }
        return;
    }

    // ---------------- compute warps
    const int lx = lane % a.g.LX;
    const int wy = lane / a.g.LX;
    const int rowi = warp * a.g.WY + wy;
    const int ry = rowi % a.g.TY, rz = rowi / a.g.TY;
    const int TXB = a.TXB, TYB = a.TYB;

    unsigned long long lst[RB];
#pragma unroll
    for (int r = 0; r < RB; r++) lst[r] = KEY_MAX;

    int it = 0;
    for (int tile = tile_begin; tile < tile_end; tile++) {
        float acc[RB][XT];
#pragma unroll
        for (int r = 0; r < RB; r++)
#pragma unroll
            for (int x = 0; x < XT; x++) acc[r][x] = 0.0f;

        for (int p = 0; p < a.P; p++, it++) {
            const int s = it % a.nstage;
            mbar_wait(&full[s], (it / a.nstage) & 1);
            const unsigned char* st = smem + static_cast<size_t>(s) * a.stage_bytes;
            const float* rec = reinterpret_cast<const float*>(st) + (rz * TYB + ry) * TXB + lx * XT;
            const float4* w4 = reinterpret_cast<const float4*>(st + a.stage_rec_bytes);
#pragma unroll 1
            for (int vz = 0; vz < M; vz++) {
#pragma unroll
                for (int vy = 0; vy < M; vy++) {
                    const float* row = rec + (vz * TYB + vy) * TXB;
                    float rv[NR4 * 4];
#pragma unroll
                    for (int j = 0; j < NR4; j++) {
                        float4 t = reinterpret_cast<const float4*>(row)[j];
                        rv[4 * j + 0] = t.x;
                        rv[4 * j + 1] = t.y;
                        rv[4 * j + 2] = t.z;
                        rv[4 * j + 3] = t.w;
                    }
#pragma unroll
                    for (int vx = 0; vx < M; vx++) {
                        const int wi = ((vz * M + vy) * M + vx) * (RB / 4);
                        float4 wa = w4[wi], wb = w4[wi + 1];
                        const float wr[RB] = {wa.x, wa.y, wa.z, wa.w, wb.x, wb.y, wb.z, wb.w};
#pragma unroll
                        for (int r = 0; r < RB; r++)
#pragma unroll
                            for (int x = 0; x < XT; x++) acc[r][x] = fmaf(wr[r], rv[x + vx], acc[r][x]);
                    }
                }
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&empty[s]);
        }

        // ---------------- epilogue for this tile
        const int tx0 = (tile % a.g.ntx) * a.g.TX + lx * XT;
        const int y = ((tile / a.g.ntx) % a.g.nty) * a.g.TY + ry;
        const int z = (tile / (a.g.ntx * a.g.nty)) * a.g.TZ + rz;
        const bool row_ok = (y < a.g.ny) && (z < a.g.nz);
        const uint32_t tbase = static_cast<uint32_t>((z * a.g.ny + y) * a.g.nx + tx0);
        if constexpr (GRID) {
            if (row_ok) {
#pragma unroll
                for (int r = 0; r < RB; r++) {
                    if (r < nb) {
                        float* out = a.grid + static_cast<size_t>(slot0 + r) * a.g.nx * a.g.ny * a.g.nz + tbase;
#pragma unroll
                        for (int x = 0; x < XT; x++)
                            if (tx0 + x < a.g.nx) out[x] = acc[r][x];
                    }
                }
            }
        } else {
            // fast check: which rotations have a value at or below their warp list's 32nd-best score?
            unsigned vmask = 0;
#pragma unroll
            for (int x = 0; x < XT; x++) vmask |= (row_ok && tx0 + x < a.g.nx) ? (1u << x) : 0u;
            unsigned pend = 0;
#pragma unroll
            for (int r = 0; r < RB; r++) {
                // exact gate: a strictly better score, or a tie whose t_lin could precede the 32nd key
                const unsigned long long l31 = shfl_u64(lst[r], 31);
                const float th = key_score_bound(static_cast<uint32_t>(l31 >> 32));
                float mn = __int_as_float(0x7f800000);
#pragma unroll
                for (int x = 0; x < XT; x++) mn = ((vmask >> x) & 1u) ? fminf(mn, acc[r][x]) : mn;
                const bool any = mn < th || (mn == th && tbase < static_cast<uint32_t>(l31 & 0xffffffffu));
                pend |= (any && r < nb) ? (1u << r) : 0u;
            }
            const unsigned wpend = __reduce_or_sync(FULL, pend);
            if (wpend) {
                // slow path, only for the rotations that need it (warp-uniform branches)
#pragma unroll
                for (int r = 0; r < RB; r++) {
                    if ((wpend >> r) & 1u) {
                        unsigned long long th = shfl_u64(lst[r], 31);
#pragma unroll
                        for (int x = 0; x < XT; x++) {
                            const unsigned long long key =
                                ((vmask >> x) & 1u) ? make_key(acc[r][x], tbase + x) : KEY_MAX;
                            unsigned m = __ballot_sync(FULL, key < th);
                            while (m) {
                                const int src = __ffs(m) - 1;
                                warp_list_insert(lst[r], shfl_u64(key, src), lane);
                                th = shfl_u64(lst[r], 31);
                                m &= ~(1u << src);
                                m &= __ballot_sync(FULL, key < th);
                            }
                        }
                    }
                }
            }
        }
    }

    if constexpr (!GRID) {
        // ---------------- item end: publish bound + surviving keys of each warp list
        const int nx = a.g.nx, ny = a.g.ny, nz = a.g.nz;
#pragma unroll 1
        for (int rr = 0; rr < RB; rr++) {
            if (rr < nb) {
                const int slot = slot0 + rr;
                const unsigned long long key = lst[0];
                const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
                const unsigned long long k31 = shfl_u64(key, 31);   // this warp list's 32nd key
                // bound: k list entries pairwise farther than 2*rho apart => key(g_k) <= key of the k-th
                bool excl = (key == KEY_MAX);
                unsigned long long Tw = KEY_MAX;
                for (int j = 0; j < a.k; j++) {
                    unsigned b = __ballot_sync(FULL, !excl);
                    if (!b) break;
                    const int f = __ffs(b) - 1;
                    const unsigned long long kf = shfl_u64(key, f);
                    const uint32_t tf = static_cast<uint32_t>(kf & 0xffffffffu);
                    excl = excl || (cheb_cyc(t, tf, nx, ny, nz) <= 2 * a.rho);
                    if (j == a.k - 1) Tw = kf;
                }
                unsigned long long Tn = 0;
                if (lane == 0) {
                    const unsigned long long old = atomicMin(&a.T[slot], Tw);
                    Tn = old < Tw ? old : Tw;
                    atomicMin(&a.mu[slot], k31);
                }
                Tn = shfl_u64(Tn, 0);
                const bool wr = (key != KEY_MAX) && (key <= Tn);
                const unsigned bal = __ballot_sync(FULL, wr);
                unsigned base = 0;
                if (lane == 0 && bal) base = atomicAdd(&a.cnt[slot], static_cast<unsigned>(__popc(bal)));
                base = __shfl_sync(FULL, base, 0);
                if (wr) {
                    const unsigned pos = base + __popc(bal & ((1u << lane) - 1u));
                    if (pos < static_cast<unsigned>(a.cap)) a.cand[static_cast<size_t>(slot) * a.cap + pos] = key;
                }
            }
            const unsigned long long l0 = lst[0];
#pragma unroll
            for (int r = 0; r < RB - 1; r++) lst[r] = lst[r + 1];
            lst[RB - 1] = l0;
        }
    }
}


// ------------------------------------------------------------------ a6: per-rotation merge + greedy filter

struct MergeArgs {
    int n_slots, k, rho, cap, n_rot;
    int nx, ny, nz;
    long long unit_begin;
    const unsigned long long* cand;
    const unsigned int* cnt;
    const unsigned long long* mu;
    int force_fallback;
    void* poses;               // dock_pose [n_slots][k]
    int* fb_list;              // flagged slots
    unsigned int* fb_cnt;
    unsigned int* cand_max;    // max candidate count seen (stats)
    const unsigned char* owned;   // block sharding: units this rank docks (others: output rows untouched); nullptr = all
};

struct PoseOut {
    int32_t rot;
    int32_t t_lin;
    float score;
    uint32_t flags;
};

// One warp per rotation.  Greedy over the candidate set W: k times take the minimum key
// that is farther than rho (cyclic Chebyshev) from every earlier pick.
// W contains every warp list's keys <= the final pruning bound T >= key(g_k); the result
// equals the exact full-grid greedy when no list's last key is below the last pick
// (mu >= key(c_k): keys are unique, so a key <= a full list's last key is in that list);
// otherwise, or on candidate overflow, the rotation is flagged for the
// exact fallback (DESIGN.md §Top-k exactness).
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_merge(MergeArgs a)
{
    __shared__ unsigned long long picks_s[8][32];
    const int wl = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int slot = blockIdx.x * (blockDim.x >> 5) + wl;
    if (slot >= a.n_slots) return;
    if (a.owned && !a.owned[slot]) return;   // another rank's unit (block sharding)
    unsigned long long* picks = picks_s[wl];
    const unsigned int n_all = a.cnt[slot];
    const unsigned int n = min(n_all, static_cast<unsigned int>(a.cap));
    if (lane == 0 && a.cand_max) atomicMax(a.cand_max, n_all);
    const unsigned long long* c = a.cand + static_cast<size_t>(slot) * a.cap;
    int np = 0;
    for (int j = 0; j < a.k; j++) {
        unsigned long long best = KEY_MAX;
        for (unsigned int i = lane; i < n; i += 32) {
            const unsigned long long key = c[i];
            if (key >= best) continue;
            const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
            bool ok = true;
            for (int q = 0; q < j; q++)
                ok = ok && (cheb_cyc(t, static_cast<uint32_t>(picks[q] & 0xffffffffu), a.nx, a.ny, a.nz) > a.rho);
            if (ok) best = key;
        }
        best = warp_min_u64(best);
        if (best == KEY_MAX) break;
        if (lane == 0) picks[j] = best;
        __syncwarp();
        np++;
    }
    const bool sound = !a.force_fallback && n_all <= static_cast<unsigned int>(a.cap) && np == a.k &&
                       a.mu[slot] >= picks[a.k - 1];   // keys are unique: a key <= a list's last key is in it
    const long long unit = a.unit_begin + slot;
    PoseOut* out = reinterpret_cast<PoseOut*>(a.poses) + static_cast<size_t>(slot) * a.k;
    for (int j = lane; j < a.k; j += 32) {
        PoseOut po;
        po.rot = static_cast<int32_t>(unit % a.n_rot);
        if (j < np) {
            po.t_lin = static_cast<int32_t>(picks[j] & 0xffffffffu);
            po.score = unord_f32(static_cast<uint32_t>(picks[j] >> 32));
            po.flags = 0;
        } else {
            po.t_lin = -1;
            po.score = __int_as_float(0x7fc00000);
            po.flags = 2u;
        }
        out[j] = po;
    }
    if (!sound && lane == 0) {
        const unsigned int idx = atomicAdd(a.fb_cnt, 1u);
        a.fb_list[idx] = slot;
    }
}
#endif

// ------------------------------------------------------------------ a6': exact greedy on a full grid

struct GreedyArgs {
    const float* grid;          // [n][nz][ny][nx]  (slot order of this fallback chunk)
    const int* slots;           // output slot of each grid
    unsigned long long* picks;  // [n][k] picks so far (KEY_MAX = none)
    int n, k, rho, n_rot, round;
    int nx, ny, nz;
    long long unit_begin;
    void* poses;
    unsigned flag_bits;         // pose flags of these picks: DOCK_POSE_FALLBACK (1) on the fallback path, 0 (FFT engine)
    const unsigned* n_live;     // optional (device): grids >= *n_live are dead (device-driven fallback)
    const struct FbDyn* dyn;    // optional (device): per-call poses / unit_begin / n_rot (device-driven fallback)
};

// Per-call arguments of the device-driven fallback, uploaded with the call's inputs (the captured fallback
// graph reads them from device memory, so it stays valid across calls).
struct FbDyn {
    VoxArgs vox;                // voxelization of the flagged slots (unit_list = the chunk's slots)
    void* poses;                // the call's dock_pose output
    long long unit_begin;
    int n_rot;
    int pad_;
};

// Control block of the fallback loop: next flagged entry to process, live slots in this chunk.
struct FbCtl {
    unsigned pos;
    unsigned n_live;
};

// One round j of the paper's best-then-exclude loop over full score grids,
// spread over many CTAs per grid: every thread scans a strided share of the N^3 cells for
// the best key that is farther than rho from picks 0..j-1, and the warp minima are combined
// with one 64-bit atomicMin per warp into picks[g][j].
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_greedy_round(GreedyArgs a)
{
    const int ctas_per_grid = gridDim.x / a.n;
    const int gi = blockIdx.x / ctas_per_grid, part = blockIdx.x % ctas_per_grid;
    if (a.n_live && gi >= static_cast<int>(*a.n_live)) return;
    const float* S = a.grid + static_cast<size_t>(gi) * a.nx * a.ny * a.nz;
    const uint32_t ncell = static_cast<uint32_t>(a.nx) * a.ny * a.nz;
    unsigned long long* pk = a.picks + static_cast<size_t>(gi) * a.k;
    const int j = a.round;
    uint32_t prev[32];
    for (int q = 0; q < j; q++) prev[q] = static_cast<uint32_t>(pk[q] & 0xffffffffu);
    if (j > 0 && pk[j - 1] == KEY_MAX) return;   // fewer than j picks possible
    unsigned long long best = KEY_MAX;
    const uint32_t stride = static_cast<uint32_t>(ctas_per_grid) * blockDim.x;
    float best_s = __int_as_float(0x7f800000);   // score of `best` (float compare first: -0 == +0, no NaN)
    auto consider = [&](uint32_t t, float sv) {
        if (sv > best_s) return;
        const unsigned long long key = make_key(sv, t);
        if (key >= best) return;
        bool ok = true;
        for (int q = 0; q < j; q++) ok = ok && (cheb_cyc(t, prev[q], a.nx, a.ny, a.nz) > a.rho);
        if (ok) {
            best = key;
            best_s = sv;
        }
    };
    // four independent loads in flight per thread (the scan is bandwidth-, not compute-bound)
    uint32_t t = part * blockDim.x + threadIdx.x;
    for (; t + 3 * stride < ncell; t += 4 * stride) {
        const float s0 = S[t], s1 = S[t + stride], s2 = S[t + 2 * stride], s3 = S[t + 3 * stride];
        consider(t, s0);
        consider(t + stride, s1);
        consider(t + 2 * stride, s2);
        consider(t + 3 * stride, s3);
    }
    for (; t < ncell; t += stride) consider(t, S[t]);
    best = warp_min_u64(best);
    if ((threadIdx.x & 31) == 0 && best != KEY_MAX) atomicMin(&pk[j], best);
}
#endif

// Write the fallback poses (flag DOCK_POSE_FALLBACK) once all rounds are done.
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_greedy_emit(GreedyArgs a)
{
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    const int n_eff = a.n_live ? min(a.n, static_cast<int>(*a.n_live)) : a.n;
    if (i >= n_eff * a.k) return;
    const int gi = i / a.k, j = i % a.k;
    void* poses = a.dyn ? a.dyn->poses : a.poses;
    const long long unit_begin = a.dyn ? a.dyn->unit_begin : a.unit_begin;
    const int n_rot = a.dyn ? a.dyn->n_rot : a.n_rot;
    const unsigned long long key = a.picks[static_cast<size_t>(gi) * a.k + j];
    const int slot = a.slots[gi];
    const long long unit = unit_begin + slot;
    PoseOut po;
    po.rot = static_cast<int32_t>(unit % n_rot);
    if (key != KEY_MAX) {
        po.t_lin = static_cast<int32_t>(key & 0xffffffffu);
        po.score = unord_f32(static_cast<uint32_t>(key >> 32));
        po.flags = a.flag_bits;
    } else {
        po.t_lin = -1;
        po.score = __int_as_float(0x7fc00000);
        po.flags = a.flag_bits | 2u;
    }
    reinterpret_cast<PoseOut*>(poses)[static_cast<size_t>(slot) * a.k + j] = po;
}
#endif

// ------------------------------------------------------------------ device-driven fallback loop
//
// The exact fallback runs as a CUDA graph: k_fb_init sets the loop condition from the
// device-side flag count k_merge produced, and a conditional WHILE node repeats
//   k_fb_chunk -> voxelize -> correlation (GRID epilogue) -> greedy rounds -> k_fb_advance
// over chunks of `ch` flagged slots.  No host synchronisation is needed whatever the count.
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_fb_init(cudaGraphConditionalHandle h, const unsigned int* fb_cnt, FbCtl* ctl)
{
    ctl->pos = 0;
    ctl->n_live = 0;
    cudaGraphSetConditional(h, *fb_cnt > 0u ? 1u : 0u);
}
__global__ void k_fb_chunk(const unsigned int* fb_cnt, const int* fb_list, FbCtl* ctl, int* slots, int ch)
{
    const unsigned pos = ctl->pos, cnt = *fb_cnt;
    const unsigned n = cnt > pos ? min(static_cast<unsigned>(ch), cnt - pos) : 0u;
    for (int i = threadIdx.x; i < ch; i += blockDim.x) slots[i] = i < static_cast<int>(n) ? fb_list[pos + i] : 0;
    if (threadIdx.x == 0) ctl->n_live = n;
}
// host-loop variants (diagnostic mode, no conditional handle)
__global__ void k_fb_init_plain(FbCtl* ctl)
{
    ctl->pos = 0;
    ctl->n_live = 0;
}
__global__ void k_fb_advance_plain(FbCtl* ctl, int ch) { ctl->pos += static_cast<unsigned>(ch); }
__global__ void k_fb_advance(cudaGraphConditionalHandle h, const unsigned int* fb_cnt, FbCtl* ctl, int ch)
{
    const unsigned pos = ctl->pos + static_cast<unsigned>(ch);
    ctl->pos = pos;
    cudaGraphSetConditional(h, pos < *fb_cnt ? 1u : 0u);
}
#endif

#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_fill_u64(unsigned long long* p, size_t n, unsigned long long v)
{
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < n;
         i += static_cast<size_t>(gridDim.x) * blockDim.x)
        p[i] = v;
}
#endif

// ------------------------------------------------------------------ input staging

// One probe's atoms in the gather table: source pointers (device memory: the caller's buffers or the
// uploaded staging copy of host arrays), atom count, destination offset.
struct ProbeSrc {
    const double* xyz;   // [n][3]
    const float* coef;   // [n][P]
    int n, off;
};

// Gather all probes' atoms into contiguous xyz [na][3] / coef [na][P] (one launch instead of two
// copies per probe).
#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_gather_probes(const ProbeSrc* __restrict__ tab, int n_probes, int P, double* __restrict__ xyz,
                                float* __restrict__ coef)
{
    const int i = blockIdx.x;
    if (i >= n_probes) return;
    const ProbeSrc t = tab[i];
    for (int j = threadIdx.x; j < 3 * t.n; j += blockDim.x) xyz[3 * static_cast<size_t>(t.off) + j] = t.xyz[j];
    for (int j = threadIdx.x; j < P * t.n; j += blockDim.x)
        coef[static_cast<size_t>(P) * t.off + j] = t.coef[j];
}
#endif

// ------------------------------------------------------------------ per-call state reset

#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_reset(unsigned long long* T, unsigned long long* mu, unsigned int* cnt, int n,
                        unsigned int* fb_cnt, unsigned int* cand_max, unsigned int* ksum)
{
    int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i < n) {
        T[i] = KEY_MAX;
        mu[i] = KEY_MAX;
        cnt[i] = 0;
    }
    if (i == 0) {
        *fb_cnt = 0;
        *cand_max = 0;
        *ksum = 0;
    }
}
#endif

}  // namespace dk

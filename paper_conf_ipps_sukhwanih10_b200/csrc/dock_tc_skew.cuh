// dock_tc_skew.cuh -- tcgen05 engine, row-skewed schedule (variants 5 and 6).
//
// Same implicit GEMM and PAIR bf16x3 scheme as k_corr_tc (dock_tc.cuh: 128 rotations x 128
// translations of one receptor x-row per MMA, K = (vz, vy, vx, 8 bf16)), but the Q accumulator rows
// of a tile are skewed by one weight stage each: in super-step g the single issuing thread runs
// stage g of row 0, stage g-1 of row 1, ..., stage g-Q+1 of row Q-1.  Rows therefore finish one
// super-step apart and restart one super-step after they finish, so the epilogue drains and scores
// row q (per-row tm_full/tm_empty barriers) while the tensor pipe keeps working on the other rows --
// the TMEM drain bubble of the unskewed schedule (one accumulator set, all rows finishing together)
// disappears without giving up the 4-fold reuse of every weight stage.
//
// The receptor boxes are staged per z-plane (one TMA box per (tile, plane), separate full/empty
// barriers), so plane p of the next tile loads as soon as the last row has used plane p of this one:
// the skew lengthens the lifetime of a box, plane granularity more than gives that back.
#pragma once
#include "dock_tc.cuh"

namespace tc {

// One 32-value chunk of scores (rotation of this thread, translations tbase + c0 + j) into the
// per-thread exact top-LIST list; GRID writes the chunk to the score grid instead.
template <bool GRID>
__device__ __forceinline__ void epi_chunk(const uint32_t (&v)[32], unsigned long long (&lst)[LIST], float& th,
                                          uint32_t& th_t, uint32_t tbase, int c0, int jmax, float* grid_row)
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
        // exact gate: a strictly better score, or a tie that could carry a smaller t_lin
        if (mn < th || (mn == th && tbase + c0 < th_t)) {
            uint32_t msk = 0;
#pragma unroll
            for (int j = 0; j < 32; j++) msk |= (__uint_as_float(v[j]) <= th && j < jmax) ? (1u << j) : 0u;
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

// Item end: bound T_w from k list entries pairwise farther than 2*rho apart, then
// publish bound, mu and the keys <= T (k_merge finishes the greedy).
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

// z-plane stride of the skewed kernels' receptor boxes (TMA destinations must be 128-B aligned)
__host__ __device__ constexpr uint32_t plane_stride(int m, int q)
{
    return (static_cast<uint32_t>(q + m - 1) * static_cast<uint32_t>(pair_txb(m)) * 16u + 127u) / 128u * 128u;
}

template <int M, int Q, int NBUF, bool GRID>
__global__ void __launch_bounds__(NTHREADS, 1) k_corr_tc_skew(const __grid_constant__ CUtensorMap tmap,
                                                               const __grid_constant__ CUtensorMap tmap_pair,
                                                               const TcArgs a)
{
    constexpr int KS = KSTEPS;
    constexpr unsigned STAGE = KS * WCHUNK;
    constexpr int MXP = (M + 1) / 2, MXQ = (M + 3) / 4;
    constexpr int S1 = M * M * MXP, S1P = (S1 + KS - 1) / KS * KS;   // pass-1 K-steps (real, padded)
    constexpr int S2 = M * M * MXQ, S2P = (S2 + KS - 1) / KS * KS;   // pass-2 K-steps
    constexpr int NS1 = S1P / KS, NS = NS1 + S2P / KS;               // weight stages per tile
    constexpr int KP1 = MXP * M, KP2 = MXQ * M;                      // K-steps per z-plane
    constexpr uint32_t ROW16 = static_cast<uint32_t>(pair_txb(M)) * 16u;
    constexpr uint32_t PLANE = static_cast<uint32_t>(Q + M - 1) * ROW16;   // bytes of one z-plane box
    constexpr uint32_t PSTRIDE = plane_stride(M, Q);                      // 128-B aligned TMA destinations
    static_assert(Q * NBUF * NT <= 512, "TMEM has 512 columns");
    static_assert(NS >= Q, "the skew needs at least Q stages per tile");
    extern __shared__ __align__(1024) unsigned char smem[];
    __shared__ uint64_t bars[4 * DOCK_MAX_M + 2 * WSTAGES + 2 * 4];
    __shared__ uint32_t tmem_base_s;
    uint64_t* main_full = bars;
    uint64_t* main_empty = bars + DOCK_MAX_M;
    uint64_t* pair_full = bars + 2 * DOCK_MAX_M;
    uint64_t* pair_empty = bars + 3 * DOCK_MAX_M;
    uint64_t* w_full = bars + 4 * DOCK_MAX_M;
    uint64_t* w_empty = w_full + WSTAGES;
    uint64_t* tm_full = w_empty + WSTAGES;   // [NBUF][Q]
    uint64_t* tm_empty = tm_full + 4;        // [NBUF][Q]

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int block = blockIdx.x / a.G, region = blockIdx.x % a.G;
    const int tile_begin = region * a.tiles_per_region;
    const int tile_end = min(a.ntiles, tile_begin + a.tiles_per_region);
    const int n_tiles = tile_end - tile_begin;
    unsigned char* main_smem = smem;
    unsigned char* pair_smem = smem + a.rec_stage_bytes;
    unsigned char* w_smem = smem + 2 * a.rec_stage_bytes;

    if (threadIdx.x == 0) {
        for (int i = 0; i < M; i++) {
            dk::mbar_init(&main_full[i], 1);
            dk::mbar_init(&main_empty[i], 1);
            dk::mbar_init(&pair_full[i], 1);
            dk::mbar_init(&pair_empty[i], 1);
        }
        for (int i = 0; i < a.wstages; i++) {
            dk::mbar_init(&w_full[i], 1);
            dk::mbar_init(&w_empty[i], 1);
        }
        for (int i = 0; i < NBUF * Q; i++) {
            dk::mbar_init(&tm_full[i], 1);
            dk::mbar_init(&tm_empty[i], a.nepi);
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
    long long tw0 = 0, tw1 = 0, tw2 = 0, tstart = tr ? clock64() : 0;
    if (n_tiles > 0) {
        if (warp == 0) {
            // ------------------------------------------------ TMA producer (one thread)
            // In stage order: the z-planes a stage is the first to read (after the previous tile's last
            // reader released them), then the stage's weights into the ring.
            if (elect_one()) {
                dk::prefetch_tmap(&tmap);
                dk::prefetch_tmap(&tmap_pair);
                const unsigned char* wsrc = a.W + static_cast<size_t>(block) * a.nsteps * WCHUNK;
                int ws = 0, wph = 0, wuse = 0;
                int tx = tile_begin % a.ntx, ty = (tile_begin / a.ntx) % a.nty, tz = tile_begin / (a.ntx * a.nty);
                for (int ti = 0; ti < n_tiles; ti++) {
                    for (int st = 0; st < NS; st++) {
#pragma unroll
                        for (int p = 0; p < M; p++) {
                            const bool m1 = st < NS1 && (p * KP1) / KS == st;
                            const bool m2 = st >= NS1 && (p * KP2) / KS == st - NS1;
                            if (m1 || m2) {
                                uint64_t* full = m1 ? &main_full[p] : &pair_full[p];
                                if (ti > 0) twait(m1 ? &main_empty[p] : &pair_empty[p], (ti - 1) & 1, tr, tw1);
                                dk::mbar_arrive_expect_tx(full, PLANE);
                                tma_load_5d((m1 ? main_smem : pair_smem) + p * PSTRIDE, m1 ? &tmap : &tmap_pair, 0,
                                            tx * NT, ty * Q, tz + p, 0, full);
                            }
                        }
                        if (wuse >= a.wstages) twait(&w_empty[ws], wph ^ 1, tr, tw0);
                        dk::mbar_arrive_expect_tx(&w_full[ws], STAGE);
                        dk::bulk_load(w_smem + static_cast<size_t>(ws) * STAGE,
                                      wsrc + static_cast<size_t>(st) * KS * WCHUNK, STAGE, &w_full[ws]);
                        wuse++;
                        if (++ws == a.wstages) {
                            ws = 0;
                            wph ^= 1;
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
                if (tr) {
                    atomicAdd(&a.trace[TR_PROD_TOTAL], static_cast<unsigned long long>(clock64() - tstart));
                    atomicAdd(&a.trace[TR_PROD_WEMPTY], static_cast<unsigned long long>(tw0));
                    atomicAdd(&a.trace[TR_PROD_REMPTY], static_cast<unsigned long long>(tw1));
                    atomicAdd(&a.trace[TR_CTAS], 1ull);
                    atomicAdd(&a.trace[TR_TILES], static_cast<unsigned long long>(n_tiles));
                }
            }
            __syncwarp();
        } else if (warp == 1) {
            // ------------------------------------------------ MMA issue (one thread), skewed rows
            constexpr uint32_t idesc = umma_idesc(ROT, NT);
            const uint64_t dA0 = umma_desc(dk::smem_u32(w_smem), ROT * 16, 128);
            const uint64_t dB0 = umma_desc(dk::smem_u32(main_smem), 16, 128);
            const uint64_t dP0 = umma_desc(dk::smem_u32(pair_smem), 32, 128);
            if (elect_one()) {
                uint32_t wsq[Q];   // ring slot of each row's next stage (rows walk the same stage sequence)
#pragma unroll
                for (int q = 0; q < Q; q++) wsq[q] = 0;
                uint32_t wph0 = 0;   // ring phase of row 0 (the first reader of every stage)
                const uint32_t nws = static_cast<uint32_t>(a.wstages);
                for (int t = 0; t <= n_tiles; t++) {
#pragma unroll
                    for (int s = 0; s < NS; s++) {
                        if (t == n_tiles && s >= Q - 1) break;   // the last tile's trailing rows are done
#pragma unroll
                        for (int qq = 0; qq < Q; qq++) {
                            // row q = s restarts (new tile) in super-step s < Q: issue it after the other rows,
                            // so the epilogue has those MMAs' time to release the row's accumulator
                            const int q = s < Q ? (qq < s ? qq : (qq < Q - 1 ? qq + 1 : s)) : qq;
                            const int ls = s >= q ? s - q : s - q + NS;   // this row's stage (compile time)
                            const int tt = s >= q ? t : t - 1;            // and tile
                            if (tt < 0 || tt >= n_tiles) continue;
                            const int buf = tt % NBUF, use = tt / NBUF;
                            if (q == 0) {
                                twait(&w_full[wsq[0]], wph0, tr, tw1);
#pragma unroll
                                for (int p = 0; p < M; p++) {
                                    if (ls < NS1 && (p * KP1) / KS == ls) twait(&main_full[p], tt & 1, tr, tw2);
                                    if (ls >= NS1 && (p * KP2) / KS == ls - NS1) twait(&pair_full[p], tt & 1, tr, tw2);
                                }
                            }
                            if (ls == 0 && use > 0) twait(&tm_empty[buf * Q + q], (use - 1) & 1, tr, tw0);
                            tc_fence_after();
                            const uint32_t dcol = tmem + static_cast<uint32_t>((buf * Q + q) * NT);
                            const uint64_t da0 = dA0 + ((wsq[q] * STAGE) >> 4);
#pragma unroll
                            for (int ks = 0; ks < KS; ks++) {
                                const uint64_t db =
                                    ls < NS1 ? dB0 + ((pair_off1(M, ls * KS + ks, ROW16, PSTRIDE) + q * ROW16) >> 4)
                                             : dP0 + ((pair_off2(M, (ls - NS1) * KS + ks, ROW16, PSTRIDE) + q * ROW16) >> 4);
                                umma_bf16(dcol, da0 + ((ks * WCHUNK) >> 4), db, idesc, (ls == 0 && ks == 0) ? 0u : 1u);
                            }
                            if (q == Q - 1) {   // last reader of this stage and of the planes it finishes
                                umma_commit(&w_empty[wsq[q]]);
#pragma unroll
                                for (int p = 0; p < M; p++) {
                                    if (ls < NS1 && ((p + 1) * KP1 - 1) / KS == ls) umma_commit(&main_empty[p]);
                                    if (ls >= NS1 && ((p + 1) * KP2 - 1) / KS == ls - NS1) umma_commit(&pair_empty[p]);
                                }
                            }
                            if (ls == NS - 1) umma_commit(&tm_full[buf * Q + q]);
                            if (++wsq[q] == nws) {
                                wsq[q] = 0;
                                if (q == 0) wph0 ^= 1;
                            }
                        }
                    }
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
            // Warp (quarter, class cls): TMEM lanes of its quarter (lane = rotation); rows in the order
            // they finish; within row q the 32-column chunks c = (q + cls + j * nclass) mod 4 (diagonal
            // classes).  A row is released right after its last chunk is in registers.
            const int quarter = warp & 3;
            const int cls = (warp - 2) >> 2;
            const int nclass = a.nepi >> 2;
            constexpr int NCH = NT / 32;
            const int r = quarter * 32 + lane;
            const int slot = block * ROT + r;
            const bool rot_ok = slot < a.n_slots;
            unsigned long long lst[LIST];
#pragma unroll
            for (int i = 0; i < LIST; i++) lst[i] = KEY_MAX;
            float th = __int_as_float(0x7f800000);
            uint32_t th_t = 0xffffffffu;
            int tx = tile_begin % a.ntx, ty = (tile_begin / a.ntx) % a.nty, tz = tile_begin / (a.ntx * a.nty);
            for (int ti = 0; ti < n_tiles; ti++) {
                const int buf = ti % NBUF, use = ti / NBUF;
                const int x0 = tx * NT;
                for (int q = 0; q < Q; q++) {
                    twait(&tm_full[buf * Q + q], use & 1, tr, tw0);
                    tc_fence_after();
                    if (a.dbg == 1) {   // diagnostic: no TMEM drain
                        __syncwarp();
                        if (lane == 0) dk::mbar_arrive(&tm_empty[buf * Q + q]);
                        continue;
                    }
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
                        if (j == NCH / nclass - 1) {
                            tc_fence_before();
                            __syncwarp();
                            if (lane == 0) dk::mbar_arrive(&tm_empty[buf * Q + q]);
                        }
                        if (!row_ok || a.dbg == 2) continue;
                        epi_chunk<GRID>(v, lst, th, th_t, tbase, c0, min(32, a.nx - x0 - c0),
                                        GRID ? a.grid + static_cast<size_t>(slot) * a.nx * a.ny * a.nz + tbase : nullptr);
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
                if (rot_ok) epi_publish(lst, slot, a);
            }
        }
    }
    tc_fence_before();
    __syncthreads();
    if (warp == 1) asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 512;" ::"r"(tmem));
}

}  // namespace tc

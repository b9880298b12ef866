// dock.cu -- host implementation of the C ABI in include/dock.h (libdock.so).
//
// Owns the device memory layout (cyclic-halo padded receptor, TMA descriptors,
// per-call scratch), validates arguments, plans launches and runs
//   reset -> k_voxelize -> k_corr<M, top-k> -> k_merge [-> exact fallback]
// on the context's stream.  Citations "P:L.." point into PAPER.md.
#include <cuda.h>
#include <cuda_runtime.h>
#include <cudaTypedefs.h>

#include <algorithm>
#include <cmath>
#include <cstdarg>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <new>
#include <vector>

#include "dock.h"
#include "dock_kernels.cuh"
#include "dock_tc.cuh"
#include "dock_sparse.cuh"
#include "dock_launch.h"
#include "dock_fft.h"

static_assert(sizeof(dock_pose) == 16, "dock_pose must be 16 bytes");
static_assert(sizeof(dk::PoseOut) == sizeof(dock_pose), "kernel pose layout mismatch");

namespace {

constexpr int kSmemLimit = 227 * 1024;

struct DevBuf {
    void* p = nullptr;
    size_t cap = 0;
};

struct TcPlan {                // per-(variant, probe size) plan of the tcgen05 engine
    bool ok = false;
    CUtensorMap tmap, tmap_pair;   // (hi,lo) receptor copy and PAIR copy (Rhi(x), Rhi(x+1))
    CUtensorMap tmap_b;            // variant 1: main half-box B (z planes [mh, m)); variant 1's tmap covers [0, mh)
    int box_bytes_b = 0, rec_off_b = 0;
    int ntt = 0, q = 0, ntx = 0, nty = 0, ntiles = 0;   // translations per row, rows per tile, tile counts
    int S1 = 0, S1p = 0, S2 = 0, S2p = 0;                // variant 1: pass-1 / pass-2 K-steps (real, padded)
    int box_bytes = 0, box_bytes_pair = 0, rec_stage_bytes = 0, n_rec_stages = 0, smem = 0, nsteps = 0, wstages = 0;
    int TXBP = 0;              // variant 1: x extent of the pair box (the main box uses TXB of make_tc_plan)
};

struct SpPlan {                // per-probe-size plan of the sparse-ligand engine (dock_sparse.cuh)
    bool ok = false;
    int xts = 0, TX = 0, ntx = 0, nty = 0, TXB = 0, TYB = 0, slot_words = 0, box_bytes = 0;
    int GXp = 0, GYp = 0, GZp = 0;   // padded atom-grid extents (cyclic halo materialised)
};

enum EngineKind { ENG_FFMA = 1, ENG_TC = 2, ENG_FFT = 3, ENG_SPARSE = 4 };

struct MPlan {                 // per-probe-size launch plan
    bool ok = false;
    CUtensorMap tmap;
    int TXB = 0, TYB = 0, TZB = 0;
    int stage_rec_bytes = 0, stage_bytes = 0, nstage = 0, smem = 0;
};

}  // namespace

struct dock_ctx {
    int device = 0;
    cudaStream_t stream = nullptr;
    bool own_stream = false;
    int nx = 0, ny = 0, nz = 0, P = 0, m_max = 0;
    double spacing = 0.0;   // h exactly as given (the kernel divides by it in FP64, like the oracle)
    int n_sms = 148;
    double l2_bytes = 0;
    dk::Geo geo{};
    float* d_rec = nullptr;
    float* d_w = nullptr;      // [P] weights
    float* d_eye = nullptr;    // [P][P] identity (per-term grids)
    float* d_ones = nullptr;   // [P] ones (unweighted voxel export)
    MPlan plan[DOCK_MAX_M + 1];
    std::vector<unsigned char> probe_dev;   // [2 n_probes] device-memory flags (xyz, coef) of the probes of
                                            // the current call, set by validate_probes for stage_inputs
    // tcgen05 engine
    int engine = 0;            // DOCK_TUNE_ENGINE: 0 auto, 1 FFMA, 2 tensor cores, 3 FFT (comparison engine)
    DockFft* fft = nullptr;    // FFT engine state (receptor transform, plans, work buffers), created on first use
    int engine_last = 0;
    int tc_variant = 0;        // DOCK_TUNE_TC_VARIANT: 0 auto, 1 resident boxes (P <= 4), 2 streamed planes
    int tc_chunk = 0;          // DOCK_TUNE_TC_CHUNK: tiles per scheduled chunk (variant 1), 0 = auto
    unsigned long long* d_sched = nullptr;   // [1 + 2 n_sms] dynamic tile scheduler counters (self-resetting)
    int tc_variant_last = 0;
    int tc_m_last = 0;
    int tc_ksteps_last = 0;    // K-steps (of 16) per translation row in the last tcgen05 launch
    int tc_nepi = 0;           // epilogue warps (0 = tc::NEPI_MAX)
    int tc_sched = 0;          // DOCK_TUNE_TC_SCHEDULE: 0 occupancy tables + clustering (m <= 4), 1 occupancy
                               // tables over consecutive units, 2 dense (every K-step)
    int tc_blocks_last = 0;
    bool tc_perm_on = false;   // the main pass's variant-1 blocks use the clustering permutation    // rotation blocks of the last variant-1 launch (executed K-step statistics)
    uint16_t* d_rec_tc = nullptr;     // [g][Zp][Yp][Xp][8] bf16 (hi_0..3, lo_0..3)
    uint16_t* d_rec_pair = nullptr;   // [g][Zp][Yp][Xp][8] bf16 (hi_0..3(X), hi_0..3(X+1))
    int tc_Gch = 0, tc_Xp = 0, tc_Yp = 0, tc_Zp = 0;
    int tcs_ntt = 128;         // variant 2 translations per MMA row, chosen for nx
    TcPlan tcplan[3][DOCK_MAX_M + 1];   // [variant][m]
    DevBuf Wtc;
    // variant 1 occupancy schedule of the main pass / of the fallback: K-step tables, source steps, per-block
    // (stages, first pair entry), clustering permutation and unit masks
    DevBuf tc_ksrc, tc_kinfo, tc_perm, tc_umask, tc_sorted, fb_ksrc, fb_kinfo, fb_umask, tc_seg, tc_pref;
    int shard_rank = 0, shard_world = 1;   // DOCK_TUNE_SHARD: block sharding of the variant-1 block order
    int tc_nblk_local = -1;    // blocks of the last main pass this rank docks (-1: all)
    DevBuf tc_blkmap, tc_owned;
    int sp_bound_every = 2;    // sparse engine: columns between global-bound refreshes (0 / 1 / 2 / 4 / 8 -> c64 0.517 / 0.457 /
                               // 0.441 / 0.477 / 0.517 ms, large shard 36.0 / 35.3 / 33.2 / 32.8 / 35.6 ms); DOCK_SP_BOUND_EVERY overrides
    int tc_seg_cost = 8;       // per-tile cost of a chunk beyond its ring stages, in ring stages (prod: 0 / 3 / 6 /
                               // 9 / 12 / 24 -> 12.20 / 11.79 / 11.40 / 11.35 / 11.48 / 11.84 ms); DOCK_TC_SEG_COST
                               // (environment) overrides it
    // diagnostics (environment, read at init): DOCK_TC_TRACE=1 prints per-role cycle counters of every
    // tcgen05 launch to stderr
    unsigned long long* d_trace = nullptr;
    // per-call scratch (grow-only)
    DevBuf xyz, coef, off, rot, Lw, T, mu, cnt, cand, poses, fb_list, grid, slots, units, Lw_fb, picks;
    int* d_small = nullptr;    // [0] status bits (sticky until the next sync point), [1] fb_cnt, [2] cand_max,
                               // [3] K-steps per tile summed over the blocks of the last variant-1 launch
    int* h_small = nullptr;    // pinned mirror, written by the async copy at the end of every call
    void* h_stage = nullptr;   // pinned scratch of the synchronous FFT comparison engine
    size_t h_stage_cap = 0;
    // pinned staging ring for the per-call inputs: a slot is rewritten only after the H2D copy that last
    // read it has executed (its event), so calls never wait for the GPU to drain
    struct Stage {
        void* h = nullptr;
        size_t cap = 0;
        cudaEvent_t ev = nullptr;
        bool live = false;
    } stage[3];
    int stage_next = 0;
    // asynchronous calls: end-of-call event (status copied to h_small), unsynced flag
    cudaEvent_t ev_done = nullptr;
    bool unsynced = false;
    // device-driven exact fallback (a CUDA graph with a WHILE node over chunks of flagged slots)
    cudaStream_t cap_stream = nullptr, cap_stream2 = nullptr;   // private capture streams
    cudaGraphExec_t fb_exec = nullptr;
    unsigned char fb_key[256] = {0};
    int fb_host_loop = 0;   // DOCK_FB_HOST_LOOP=1 (environment): fallback from a host loop instead of the graph
    DevBuf fb_grid, fb_Lw, fb_W, fb_picks, fb_slots, fb_ctl, fb_groups;
    // sparse-ligand engine: plans, atom grids G_a of the call, occupied-voxel term tables
    SpPlan spplan[DOCK_MAX_M + 1][6];   // [m][xts]
    DevBuf sp_G, sp_tv, sp_ts, sp_nt, sp_dw, sp_slot_atoms;
    CUtensorMap sp_tmap;
    int sp_natoms_last = 0;           // atom grids of the last sparse call
    int sp_tx_last = 0, sp_zt_last = 0;
    double sp_terms_last = 0;         // occupied voxels summed over the units of the last sparse call
    // tuning
    int regions_override = 0;
    int force_fallback = 0;
    int cand_cap = 1024;
    // stats
    int regions_last = 0;
    int64_t items_last = 0, fallback_last = 0, cand_max_last = 0, kernels_last = 0;
    cudaEvent_t ev_corr[2] = {nullptr, nullptr};   // bracket the k_corr launch of dock_probe_batch
    bool ev_corr_valid = false;
    bool dead = false;
    char err[512] = {0};
};

namespace {

dock_status fail(dock_ctx* c, dock_status s, const char* fmt, ...)
{
    if (c) {
        va_list ap;
        va_start(ap, fmt);
        vsnprintf(c->err, sizeof(c->err), fmt, ap);
        va_end(ap);
        if (s == DOCK_E_CUDA) c->dead = true;
    }
    return s;
}

#define CU(call)                                                                                        \
    do {                                                                                                \
        cudaError_t e_ = (call);                                                                        \
        if (e_ != cudaSuccess) {                                                                        \
            return fail(ctx, e_ == cudaErrorMemoryAllocation ? DOCK_E_OOM : DOCK_E_CUDA, "%s: %s (%s:%d)", \
                        #call, cudaGetErrorString(e_), __FILE__, __LINE__);                             \
        }                                                                                               \
    } while (0)

#define TRY(expr)                          \
    do {                                   \
        dock_status s_ = (expr);           \
        if (s_ != DOCK_OK) return s_;      \
    } while (0)

// 0 = host memory (pageable or pinned), 1 = device memory of `device` (or managed), -1 = device memory of
// another device (the kernels of this context cannot use it)
int ptr_kind(const void* p, int device)
{
    if (!p) return 0;
    cudaPointerAttributes at;
    if (cudaPointerGetAttributes(&at, p) != cudaSuccess) {
        cudaGetLastError();
        return 0;
    }
    if (at.type == cudaMemoryTypeManaged) return 1;
    if (at.type == cudaMemoryTypeDevice) return at.device == device ? 1 : -1;
    return 0;
}

bool is_device_ptr(const void* p)
{
    if (!p) return false;
    cudaPointerAttributes at;
    if (cudaPointerGetAttributes(&at, p) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return at.type == cudaMemoryTypeDevice || at.type == cudaMemoryTypeManaged;
}

// Device-or-host classification of a caller pointer; device memory of another device is an argument error.
#define PTR_KIND(dst, p, what)                                                                           \
    do {                                                                                                 \
        int k_ = ptr_kind((p), ctx->device);                                                             \
        if (k_ < 0) return fail(ctx, DOCK_E_INVALID_ARG, "%s is device memory of another device", what); \
        dst = (k_ == 1);                                                                                 \
    } while (0)

// Next slot of the pinned staging ring (waits only for the H2D copy that last read the slot).
dock_status acquire_stage(dock_ctx* ctx, size_t bytes, dock_ctx::Stage** out)
{
    dock_ctx::Stage& st = ctx->stage[ctx->stage_next];
    ctx->stage_next = (ctx->stage_next + 1) % 3;
    if (st.live) CU(cudaEventSynchronize(st.ev));
    st.live = false;
    if (bytes > st.cap) {
        if (st.h) CU(cudaFreeHost(st.h));
        st.h = nullptr;
        st.cap = 0;
        const size_t want = std::max<size_t>(bytes + bytes / 2, 1 << 16);
        CU(cudaHostAlloc(&st.h, want, cudaHostAllocDefault));
        st.cap = want;
    }
    *out = &st;
    return DOCK_OK;
}

dock_status ensure(dock_ctx* ctx, DevBuf& b, size_t bytes)
{
    if (bytes <= b.cap) return DOCK_OK;
    if (b.p) CU(cudaFree(b.p));
    b.p = nullptr;
    b.cap = 0;
    size_t want = std::max<size_t>(bytes, 256);
    CU(cudaMalloc(&b.p, want));
    b.cap = want;
    return DOCK_OK;
}

dock_status ensure_pinned(dock_ctx* ctx, size_t bytes)
{
    if (bytes <= ctx->h_stage_cap) return DOCK_OK;
    if (ctx->h_stage) {
        CU(cudaStreamSynchronize(ctx->stream));
        CU(cudaFreeHost(ctx->h_stage));
    }
    ctx->h_stage = nullptr;
    ctx->h_stage_cap = 0;
    size_t want = std::max<size_t>(bytes, 1 << 16);
    CU(cudaHostAlloc(&ctx->h_stage, want, cudaHostAllocDefault));
    ctx->h_stage_cap = want;
    return DOCK_OK;
}

int round_up(int v, int a) { return (v + a - 1) / a * a; }

PFN_cuTensorMapEncodeTiled_v12000 encode_fn()
{
    static PFN_cuTensorMapEncodeTiled_v12000 fn = nullptr;
    if (!fn) {
        void* p = nullptr;
        cudaDriverEntryPointQueryResult q;
        if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
            q == cudaDriverEntryPointSuccess)
            fn = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(p);
        else
            cudaGetLastError();
    }
    return fn;
}

// Tile geometry: XT = 8 translations per lane along x, LX lanes per row.  LX is chosen to
// waste the fewest x translations (ties: wider rows, less halo).
dk::Geo choose_geo(int nx, int ny, int nz, int m_max)
{
    dk::Geo g{};
    g.nx = nx;
    g.ny = ny;
    g.nz = nz;
    int best = 16;
    double best_w = 1e30;
    for (int lx : {16, 8, 4}) {
        int tx = lx * dk::XT;
        int ntx = (nx + tx - 1) / tx;
        double w = double(ntx) * tx / nx;
        if (w < best_w - 1e-9) {
            best_w = w;
            best = lx;
        }
    }
    g.LX = best;
    g.WY = 32 / best;
    g.TX = best * dk::XT;
    int rows = dk::NWC * g.WY;   // 16, 32 or 64
    g.TY = rows == 16 ? 4 : 8;
    g.TZ = rows / g.TY;
    g.ntx = (nx + g.TX - 1) / g.TX;
    g.nty = (ny + g.TY - 1) / g.TY;
    g.ntz = (nz + g.TZ - 1) / g.TZ;
    g.ntiles = g.ntx * g.nty * g.ntz;
    int txb_max = round_up(g.TX + m_max - 1, 4);
    g.Xp = round_up((g.ntx - 1) * g.TX + txb_max, 4);
    g.Yp = g.nty * g.TY + m_max - 1;
    g.Zp = g.ntz * g.TZ + m_max - 1;
    return g;
}

dock_status make_plan(dock_ctx* ctx, int m)
{
    MPlan& pl = ctx->plan[m];
    if (pl.ok) return DOCK_OK;
    const dk::Geo& g = ctx->geo;
    pl.TXB = round_up(g.TX + m - 1, 4);
    pl.TYB = g.TY + m - 1;
    pl.TZB = g.TZ + m - 1;
    if (pl.TXB > 256 || pl.TYB > 256 || pl.TZB > 256)
        return fail(ctx, DOCK_E_UNSUPPORTED, "TMA box too large");
    pl.stage_rec_bytes = round_up(pl.TXB * pl.TYB * pl.TZB * 4, 128);
    pl.stage_bytes = round_up(pl.stage_rec_bytes + m * m * m * dk::RB * 4, 128);
    int ns = (kSmemLimit - 256) / pl.stage_bytes;
    ns = std::min(ns, 4);
    if (ns < 2) return fail(ctx, DOCK_E_UNSUPPORTED, "probe grid m=%d too large for the shared-memory ring", m);
    pl.nstage = ns;
    pl.smem = ns * pl.stage_bytes + 2 * ns * 8;
    auto fn = encode_fn();
    if (!fn) return fail(ctx, DOCK_E_CUDA, "cuTensorMapEncodeTiled unavailable");
    cuuint64_t dims[4] = {(cuuint64_t)g.Xp, (cuuint64_t)g.Yp, (cuuint64_t)g.Zp, (cuuint64_t)ctx->P};
    cuuint64_t strides[3] = {(cuuint64_t)g.Xp * 4, (cuuint64_t)g.Xp * g.Yp * 4, (cuuint64_t)g.Xp * g.Yp * g.Zp * 4};
    cuuint32_t box[4] = {(cuuint32_t)pl.TXB, (cuuint32_t)pl.TYB, (cuuint32_t)pl.TZB, 1};
    cuuint32_t es[4] = {1, 1, 1, 1};
    CUresult r = fn(&pl.tmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 4, ctx->d_rec, dims, strides, box, es,
                    CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                    CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (r != CUDA_SUCCESS) return fail(ctx, DOCK_E_CUDA, "cuTensorMapEncodeTiled failed (%d)", (int)r);
    pl.ok = true;
    return DOCK_OK;
}

// tcgen05 engine (dock_tc.cuh): variant 1 = one channel group, both receptor boxes resident, 128
// translations x 4 rows per tile; variant 2 = any channel count, receptor streamed one (group, z-plane)
// unit at a time, NTT in {64, 128, 160} translations per row (chosen at init for nx) x tcs_q(NTT) rows.
dock_status make_tc_plan(dock_ctx* ctx, int m, int v)
{
    TcPlan& pl = ctx->tcplan[v][m];
    if (pl.ok || !ctx->d_rec_tc || !ctx->d_rec_pair) return DOCK_OK;
    const int KS = tc::KSTEPS;
    const int budget = kSmemLimit - 512;    // static shared memory (barriers: < 400 B)
    const int stage = KS * tc::WCHUNK;
    int TXB = 0, TYB = 0, TZB = 0;
    int rec_bytes = 0;   // shared memory before the weight ring
    if (v == 1) {
        if (ctx->tc_Gch != 1) return DOCK_OK;   // one channel group only
        pl.ntt = tc::NT;
        pl.q = 4;
        TXB = tc::main_box_txb(m);
        pl.TXBP = tc::pair_box_txb(m);
        TYB = pl.q + m - 1;
        TZB = m;
        // the main box as two half-boxes (z planes [0, mh) and [mh, m)) with their own barriers: the next tile's
        // half A streams in while this tile still reads half B and the pair box (dock_tc.cuh: k_corr_tc)
        const int mh = (m + 1) / 2;
        pl.box_bytes = 16 * TXB * TYB * mh;
        pl.box_bytes_b = 16 * TXB * TYB * (m - mh);
        pl.rec_off_b = round_up(pl.box_bytes, 128);
        pl.box_bytes_pair = 16 * pl.TXBP * TYB * TZB;
        pl.rec_stage_bytes = round_up(pl.rec_off_b + pl.box_bytes_b, 128);   // offset of the pair box
        rec_bytes = pl.rec_stage_bytes + round_up(pl.box_bytes_pair, 128);
        pl.n_rec_stages = 2;   // main box + pair box
        const int MXP = (m + 1) / 2, MXQ = (m + 3) / 4;
        pl.S1 = m * m * MXP;
        pl.S1p = round_up(pl.S1, KS);
        pl.S2 = m * m * MXQ;
        pl.S2p = round_up(pl.S2, KS);
        pl.nsteps = pl.S1p + pl.S2p;
        if (rec_bytes + 3 * stage > budget) return DOCK_OK;   // not eligible for this m
    } else {
        pl.ntt = ctx->tcs_ntt;
        pl.q = tcs_q(pl.ntt);
        TXB = tc::pair_txb(m, pl.ntt);
        TYB = pl.q + m - 1;
        TZB = 1;
        pl.box_bytes = 16 * TXB * TYB;   // one z-plane
        pl.rec_stage_bytes = round_up(2 * (int)tc::stream_plane_stride(m, pl.ntt, pl.q), 1024);
        pl.n_rec_stages = 3 * pl.rec_stage_bytes + 6 * stage <= budget ? 3 : 2;
        if (pl.n_rec_stages * pl.rec_stage_bytes + 3 * stage > budget) return DOCK_OK;
        rec_bytes = pl.n_rec_stages * pl.rec_stage_bytes;
        pl.nsteps = ctx->tc_Gch * m * tc::unit_ksteps_padded(m);
    }
    if (TXB > 256 || TYB > 256 || pl.TXBP > 256) return DOCK_OK;   // TMA box limit
    pl.ntx = (ctx->nx + pl.ntt - 1) / pl.ntt;
    pl.nty = (ctx->ny + pl.q - 1) / pl.q;
    pl.ntiles = pl.ntx * pl.nty * ctx->nz;
    if ((pl.ntx - 1) * pl.ntt + std::max(TXB, pl.TXBP) > ctx->tc_Xp || pl.nty * pl.q + m - 1 > ctx->tc_Yp)
        return fail(ctx, DOCK_E_CUDA, "tcgen05 receptor padding too small");
    pl.wstages = std::min(tc::WSTAGES, (budget - rec_bytes) / stage);
    // >= 116 KB keeps one CTA per SM: every CTA allocates all 512 TMEM columns
    pl.smem = std::max(rec_bytes + pl.wstages * stage, 116 * 1024);
    auto fn = encode_fn();
    if (!fn) return fail(ctx, DOCK_E_CUDA, "cuTensorMapEncodeTiled unavailable");
    const cuuint64_t X = ctx->tc_Xp, Y = ctx->tc_Yp, Z = ctx->tc_Zp;
    cuuint64_t dims[5] = {8, X, Y, Z, (cuuint64_t)ctx->tc_Gch};
    cuuint64_t strides[4] = {16, X * 16, X * Y * 16, X * Y * Z * 16};
    cuuint32_t es[5] = {1, 1, 1, 1, 1};
    for (int which = 0; which < 3; which++) {
        const int mh = (m + 1) / 2;
        if (which == 2 && (v != 1 || m - mh == 0 || m - mh == mh)) {
            pl.tmap_b = pl.tmap;   // same half-box shape (or no second half)
            continue;
        }
        const int tzb = v != 1 ? TZB : which == 0 ? mh : which == 2 ? m - mh : TZB;
        cuuint32_t box[5] = {8, (cuuint32_t)(which == 1 && v == 1 ? pl.TXBP : TXB), (cuuint32_t)TYB, (cuuint32_t)tzb, 1};
        CUresult r = fn(which == 1 ? &pl.tmap_pair : which == 2 ? &pl.tmap_b : &pl.tmap, CU_TENSOR_MAP_DATA_TYPE_BFLOAT16, 5,
                        which == 1 ? (void*)ctx->d_rec_pair : (void*)ctx->d_rec_tc, dims, strides, box, es,
                        CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                        CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
        if (r != CUDA_SUCCESS) return fail(ctx, DOCK_E_CUDA, "cuTensorMapEncodeTiled (bf16) failed (%d)", (int)r);
    }
    pl.ok = true;
    return DOCK_OK;
}

cudaError_t launch_tc(int m, int v, bool grid, const TcPlan& pl, const tc::TcArgs& a, int nblocks, cudaStream_t st)
{
    if (v == 1) return dock_launch_tc1(m, grid, pl.tmap, pl.tmap_pair, pl.tmap_b, pl.smem, a, nblocks, st);
    return dock_launch_tcs(m, pl.ntt, grid, pl.tmap, pl.tmap_pair, pl.smem, a, nblocks, st);
}

// Regions per rotation block (tcgen05): minimise waves * (tiles per item + per-item overhead).
int choose_regions_n(const dock_ctx* ctx, int64_t n_batches, int nt)
{
    if (ctx->regions_override > 0) return std::min(ctx->regions_override, nt);
    int best = 1;
    double best_cost = 1e300;
    for (int G = 1; G <= std::min(nt, 512); G++) {
        int tpr = (nt + G - 1) / G;
        int geff = (nt + tpr - 1) / tpr;
        int64_t items = n_batches * geff;
        int64_t waves = (items + ctx->n_sms - 1) / ctx->n_sms;
        double cost = double(waves) * (tpr + 0.5);
        if (cost < best_cost - 1e-9) {
            best_cost = cost;
            best = geff;
        }
    }
    return best;
}

// Regions per rotation batch: minimise waves * (tiles per item + per-item overhead).
int choose_regions(const dock_ctx* ctx, int64_t n_batches)
{
    if (ctx->regions_override > 0) return std::min(ctx->regions_override, ctx->geo.ntiles);
    const int nt = ctx->geo.ntiles;
    int best = 1;
    double best_cost = 1e300;
    for (int G = 1; G <= std::min(nt, 256); G++) {
        int tpr = (nt + G - 1) / G;
        int geff = (nt + tpr - 1) / tpr;
        int64_t items = n_batches * geff;
        int64_t waves = (items + ctx->n_sms - 1) / ctx->n_sms;
        double cost = double(waves) * (tpr + 0.5);
        if (cost < best_cost - 1e-9) {
            best_cost = cost;
            best = geff;
        }
    }
    return best;
}

dock_status check_ctx(dock_ctx* ctx)
{
    if (!ctx) return DOCK_E_INVALID_ARG;
    if (ctx->dead) return fail(ctx, DOCK_E_CUDA, "context unusable after an earlier CUDA error");
    cudaError_t e = cudaSetDevice(ctx->device);
    if (e != cudaSuccess) return fail(ctx, DOCK_E_CUDA, "cudaSetDevice: %s", cudaGetErrorString(e));
    return DOCK_OK;
}

// Stage probes (atoms packed probe by probe) and rotations on the device.
// Returns device pointers in *xyz, *coef, *off, *rot.  With fb != nullptr the fallback's per-call
// arguments (dk::FbDyn, its vox.xyz/coef/atom_off/rot filled in here) travel in the same H2D copy and
// *d_fb receives their device address.
dock_status stage_inputs(dock_ctx* ctx, const dock_probe_desc* probes, int n_probes, const double* rot,
                         int n_rot, const double** d_xyz, const float** d_coef, const int** d_off,
                         const double** d_rot, dk::FbDyn* fb = nullptr, const dk::FbDyn** d_fb = nullptr,
                         const void* extra = nullptr, size_t extra_bytes = 0, const void** d_extra = nullptr)
{
    // One pinned staging block [fb args][off][gather table][rot (host)][host xyz][host coef] goes up in a
    // single H2D copy; one gather kernel then assembles all probes' atoms (device-resident probe arrays are
    // read in place).  The host part stays short and never waits for the GPU (staging ring).  The probes'
    // memory kinds are those validate_probes recorded for this call.
    if (ctx->probe_dev.size() != 2 * (size_t)n_probes)
        return fail(ctx, DOCK_E_INVALID_ARG, "internal: probes not validated");
    const int P = ctx->P;
    std::vector<int> off(n_probes + 1, 0);
    for (int i = 0; i < n_probes; i++) off[i + 1] = off[i] + probes[i].n_atoms;
    const int na = off[n_probes];
    bool rot_dev = false;
    PTR_KIND(rot_dev, rot, "rot");
    const size_t b_fb = fb ? (sizeof(dk::FbDyn) + 15) / 16 * 16 : 0;
    const size_t b_off = sizeof(int) * (n_probes + 1), b_tab = sizeof(dk::ProbeSrc) * std::max(n_probes, 1);
    const size_t b_rot = rot_dev ? 0 : sizeof(double) * 9 * n_rot;
    const size_t b_xyz = sizeof(double) * 3 * std::max(na, 1), b_coef = sizeof(float) * P * std::max(na, 1);
    const size_t o_off = b_fb, o_tab = o_off + (b_off + 15) / 16 * 16, o_rot = o_tab + (b_tab + 15) / 16 * 16;
    const size_t o_xyz = o_rot + (b_rot + 15) / 16 * 16, o_coef = o_xyz + (b_xyz + 15) / 16 * 16;
    const size_t o_extra = o_coef + (b_coef + 15) / 16 * 16;   // optional blob (sparse engine: group table)
    const size_t total = o_extra + extra_bytes;
    TRY(ensure(ctx, ctx->xyz, b_xyz));
    TRY(ensure(ctx, ctx->coef, b_coef));
    TRY(ensure(ctx, ctx->off, total));   // device copy of the whole staging block
    dock_ctx::Stage* stg = nullptr;
    TRY(acquire_stage(ctx, total, &stg));
    char* hs = static_cast<char*>(stg->h);
    char* ds = static_cast<char*>(ctx->off.p);
    memcpy(hs + o_off, off.data(), b_off);
    if (!rot_dev) memcpy(hs + o_rot, rot, b_rot);
    auto* tab = reinterpret_cast<dk::ProbeSrc*>(hs + o_tab);
    for (int i = 0; i < n_probes; i++) {
        const dock_probe_desc& pr = probes[i];
        dk::ProbeSrc t{};
        t.n = pr.n_atoms;
        t.off = off[i];
        if (pr.n_atoms > 0) {
            const size_t bx = sizeof(double) * 3 * pr.n_atoms, bc = sizeof(float) * P * pr.n_atoms;
            const bool xd = ctx->probe_dev[2 * i], cd = ctx->probe_dev[2 * i + 1];
            if (xd) {
                t.xyz = pr.xyz;
            } else {
                memcpy(hs + o_xyz + sizeof(double) * 3 * (size_t)off[i], pr.xyz, bx);
                t.xyz = reinterpret_cast<const double*>(ds + o_xyz) + 3 * (size_t)off[i];
            }
            if (cd) {
                t.coef = pr.coef;
            } else {
                memcpy(hs + o_coef + sizeof(float) * P * (size_t)off[i], pr.coef, bc);
                t.coef = reinterpret_cast<const float*>(ds + o_coef) + (size_t)P * off[i];
            }
        }
        tab[i] = t;
    }
    *d_rot = rot_dev ? rot : reinterpret_cast<const double*>(ds + o_rot);
    *d_xyz = static_cast<const double*>(ctx->xyz.p);
    *d_coef = static_cast<const float*>(ctx->coef.p);
    *d_off = reinterpret_cast<const int*>(ds + o_off);
    if (extra_bytes) {
        memcpy(hs + o_extra, extra, extra_bytes);
        *d_extra = ds + o_extra;
    }
    if (fb) {
        fb->vox.xyz = *d_xyz;
        fb->vox.coef = *d_coef;
        fb->vox.atom_off = *d_off;
        fb->vox.rot = *d_rot;
        memcpy(hs, fb, sizeof(dk::FbDyn));
        *d_fb = reinterpret_cast<const dk::FbDyn*>(ds);
    }
    CU(cudaMemcpyAsync(ds, hs, total, cudaMemcpyHostToDevice, ctx->stream));
    CU(cudaEventRecord(stg->ev, ctx->stream));
    stg->live = true;
    if (n_probes > 0) {
        dk::k_gather_probes<<<n_probes, 64, 0, ctx->stream>>>(reinterpret_cast<const dk::ProbeSrc*>(ds + o_tab),
                                                              n_probes, P, static_cast<double*>(ctx->xyz.p),
                                                              static_cast<float*>(ctx->coef.p));
        CU(cudaGetLastError());
        ctx->kernels_last++;
    }
    return DOCK_OK;
}

dock_status validate_probes(dock_ctx* ctx, const dock_probe_desc* probes, int n_probes, int* m_out)
{
    if (!probes || n_probes < 1) return fail(ctx, DOCK_E_INVALID_ARG, "no probes");
    int m = probes[0].m;
    ctx->probe_dev.assign(2 * (size_t)n_probes, 0);
    for (int i = 0; i < n_probes; i++) {
        const dock_probe_desc& p = probes[i];
        if (p.n_atoms < 0) return fail(ctx, DOCK_E_INVALID_ARG, "probe %d: n_atoms < 0", i);
        if (p.n_atoms > 0 && (!p.xyz || !p.coef)) return fail(ctx, DOCK_E_INVALID_ARG, "probe %d: null atoms", i);
        if (p.m < 1) return fail(ctx, DOCK_E_INVALID_ARG, "probe %d: m < 1", i);
        if (p.m > ctx->m_max || p.m > DOCK_MAX_M)
            return fail(ctx, DOCK_E_UNSUPPORTED, "probe %d: m=%d exceeds m_max=%d", i, p.m, ctx->m_max);
        if (p.m != m) return fail(ctx, DOCK_E_UNSUPPORTED, "probes of different m in one batch");
        bool xd = false, cd = false;
        PTR_KIND(xd, p.xyz, "probe xyz");
        PTR_KIND(cd, p.coef, "probe coef");
        ctx->probe_dev[2 * i] = xd;
        ctx->probe_dev[2 * i + 1] = cd;
        if (!xd && p.n_atoms > 0) {
            for (int j = 0; j < 3 * p.n_atoms; j++)
                if (!std::isfinite(p.xyz[j])) return fail(ctx, DOCK_E_INVALID_ARG, "probe %d: non-finite xyz", i);
        }
        if (!cd && p.n_atoms > 0) {
            for (int j = 0; j < ctx->P * p.n_atoms; j++)
                if (!std::isfinite(p.coef[j])) return fail(ctx, DOCK_E_INVALID_ARG, "probe %d: non-finite coef", i);
        }
    }
    *m_out = m;
    return DOCK_OK;
}

dock_status run_voxelize(dock_ctx* ctx, int m, int n_slots, int64_t unit_begin, const int* d_units, int n_rot,
                         const double* xyz, const float* coef, const int* off, const double* rot, const float* w,
                         float* Lw)
{
    dk::VoxArgs v{};
    v.xyz = xyz;
    v.coef = coef;
    v.atom_off = off;
    v.rot = rot;
    v.w = w;
    v.unit_list = d_units;
    v.unit_begin = unit_begin;
    v.n_rot = n_rot;
    v.n_slots = n_slots;
    v.P = ctx->P;
    v.m = m;
    v.spacing = ctx->spacing;
    v.Lw = Lw;
    v.status = ctx->d_small;
    int n = (n_slots + dk::RB - 1) / dk::RB * dk::RB * ctx->P;
    dk::k_voxelize<<<(n + 127) / 128, 128, 0, ctx->stream>>>(v);
    CU(cudaGetLastError());
    ctx->kernels_last++;
    return DOCK_OK;
}

dk::CorrArgs corr_args(dock_ctx* ctx, int m, int n_slots, int G, const float* Lw)
{
    const MPlan& pl = ctx->plan[m];
    dk::CorrArgs a{};
    a.g = ctx->geo;
    a.P = ctx->P;
    a.Lw = Lw;
    a.n_slots = n_slots;
    a.G = G;
    a.tiles_per_region = (ctx->geo.ntiles + G - 1) / G;
    a.nstage = pl.nstage;
    a.stage_rec_bytes = pl.stage_rec_bytes;
    a.box_bytes = pl.TXB * pl.TYB * pl.TZB * 4;
    a.stage_bytes = pl.stage_bytes;
    a.TXB = pl.TXB;
    a.TYB = pl.TYB;
    a.TZB = pl.TZB;
    return a;
}

// Score grids for n slots (GRID epilogue) into grid[n][nz][ny][nx].
dock_status run_grid(dock_ctx* ctx, int m, int n_slots, const float* Lw, float* grid)
{
    int64_t nb = (n_slots + dk::RB - 1) / dk::RB;
    int G = choose_regions(ctx, nb);
    dk::CorrArgs a = corr_args(ctx, m, n_slots, G, Lw);
    a.grid = grid;
    CU(dock_launch_ffma(m, true, ctx->plan[m].tmap, ctx->plan[m].smem, a, (int)(nb * G), ctx->stream));
    ctx->kernels_last++;
    return DOCK_OK;
}

tc::TcArgs tc_args(dock_ctx* ctx, int m, int v, int n_slots, int G, const unsigned char* W)
{
    const TcPlan& tp = ctx->tcplan[v][m];
    tc::TcArgs a{};
    a.nx = ctx->nx;
    a.ny = ctx->ny;
    a.nz = ctx->nz;
    a.ntx = tp.ntx;
    a.nty = tp.nty;
    a.ntz = ctx->nz;
    a.ntiles = tp.ntiles;
    a.G_ch = ctx->tc_Gch;
    a.n_slots = n_slots;
    a.G = G;
    a.tiles_per_region = (a.ntiles + G - 1) / G;
    a.nsteps = tp.nsteps;
    a.W = W;
    if (v == 1) {   // main pass tables unless W is the fallback's operand
        const bool fb = W == static_cast<const unsigned char*>(ctx->fb_W.p);
        a.kinfo = static_cast<const int4*>(fb ? ctx->fb_kinfo.p : ctx->tc_kinfo.p);
        a.perm = (!fb && ctx->tc_perm_on) ? static_cast<const int*>(ctx->tc_perm.p) : nullptr;
        if (!fb && ctx->tc_nblk_local >= 0) {   // block sharding
            a.blkmap = static_cast<const int*>(ctx->tc_blkmap.p);
            a.n_blocks = ctx->tc_nblk_local;
        }
    }
    a.box_bytes = tp.box_bytes;
    a.box_bytes_pair = tp.box_bytes_pair;
    a.box_bytes_b = tp.box_bytes_b;
    a.rec_off_b = tp.rec_off_b;
    a.rec_stage_bytes = tp.rec_stage_bytes;
    a.n_rec_stages = tp.n_rec_stages;
    a.wstages = tp.wstages;
    a.nepi = ctx->tc_nepi > 0 ? std::min(tc::NEPI_MAX, ctx->tc_nepi) : tc::NEPI_MAX;
    a.trace = ctx->d_trace;
    // variant 1 (one CTA per SM: >= 116 KB shared memory, all 512 TMEM columns): a persistent CTA per SM takes
    // chunks of tc_chunk tiles of one rotation block from a device counter.  Per-tile cost varies with the
    // receptor region (top-k insertions), so static splits leave SMs idle at the end (measured: CTA lifetimes
    // 1.05-2.05 ms for equal tile counts at 1008 rotations); region mode also quantises to whole waves.  A
    // forced region count (DOCK_TUNE_REGIONS) keeps region mode.
    a.chunk = 0;
    a.sched = ctx->d_sched;
    if (v == 1 && ctx->regions_override <= 0 && ctx->d_sched) {
        // auto: 16 tiles per chunk for long launches (fewer chunk hand-offs), 4 for short ones (finer load
        // balance at the tail).  Measured (kernel ms): prod (1743 tiles per CTA) 4 / 8 / 16 / 32 / 64 ->
        // 11.02 / 10.90 / 10.87 / 10.95 / 11.13; 1008 units (221 tiles per CTA) -> 1.91 / 1.94 / 1.99 / 2.00 / 2.14
        const int64_t nb = (a.blkmap ? a.n_blocks : (n_slots + tc::ROT - 1) / tc::ROT);
        const int64_t per_cta = nb * a.ntiles / std::max(1, ctx->n_sms);
        a.chunk = ctx->tc_chunk > 0 ? ctx->tc_chunk : (int)std::min<int64_t>(16, std::max<int64_t>(4, per_cta / 100));
    }
    return a;
}

// CTAs of a tensor-core launch over n_slots rotations.
int64_t tc_ctas(const tc::TcArgs& a, int n_slots, int n_sms)
{
    const int64_t n_blocks = a.blkmap ? a.n_blocks : (n_slots + tc::ROT - 1) / tc::ROT;
    if (a.chunk > 0) return std::min<int64_t>(n_sms, n_blocks * ((a.ntiles + a.chunk - 1) / a.chunk));
    return n_blocks * a.G;
}

// Variant + regions for a launch over n_slots rotations; returns false if the tensor cores can't run m.
// Auto: variant 1 where it runs with the same row width as variant 2 would use (its resident boxes
// need no per-plane synchronisation), else variant 2.
bool plan_tc_launch(dock_ctx* ctx, int m, int n_slots, int* v_out, int* G_out)
{
    const int64_t n_blocks = (n_slots + tc::ROT - 1) / tc::ROT;
    const bool ok1 = ctx->tcplan[1][m].ok, ok2 = ctx->tcplan[2][m].ok;
    int v = 0;
    if (ctx->tc_variant == 1 && ok1) v = 1;
    else if (ctx->tc_variant == 2 && ok2) v = 2;
    else if (ok1 && (ctx->tcs_ntt == tc::NT || !ok2)) v = 1;
    else if (ok2) v = 2;
    if (!v) return false;
    *v_out = v;
    *G_out = choose_regions_n(ctx, n_blocks, ctx->tcplan[v][m].ntiles);
    return true;
}

// Engine choice.  Forced: 1 FFMA, 2 tcgen05, 4 sparse ligand (DOCK_E_UNSUPPORTED when ineligible).  Auto:
// the sparse-ligand engine when it is eligible and its cost model (one gathered value per occupied voxel and
// translation) beats the dense engine's, else tcgen05 when a plan exists for m, else FFMA.
dock_status select_engine(dock_ctx* ctx, int m, bool sparse_ok, bool sparse_better, int* kind)
{
    int v = 0, G = 0;
    const bool tc_ok = plan_tc_launch(ctx, m, tc::ROT, &v, &G);
    if (ctx->engine == 2 && !tc_ok) return fail(ctx, DOCK_E_UNSUPPORTED, "tensor-core engine unavailable for m=%d", m);
    if (ctx->engine == 4 && !sparse_ok)
        return fail(ctx, DOCK_E_UNSUPPORTED, "sparse-ligand engine ineligible (atoms per probe or shared memory)");
    int k = ENG_FFMA;
    if (ctx->engine == 1) k = ENG_FFMA;
    else if (ctx->engine == 2) k = ENG_TC;
    else if (ctx->engine == 4) k = ENG_SPARSE;
    else k = (sparse_ok && sparse_better) ? ENG_SPARSE : tc_ok ? ENG_TC : ENG_FFMA;
    *kind = k;
    ctx->engine_last = k;
    if (k != ENG_TC) ctx->tc_variant_last = 0;
    return DOCK_OK;
}

// ---------------------------------------------------------------- sparse-ligand engine (dock_sparse.cuh)

dock_status make_sp_plan(dock_ctx* ctx, int m, int xts)
{
    SpPlan& pl = ctx->spplan[m][xts];
    if (pl.ok) return DOCK_OK;
    pl.xts = xts;
    pl.TX = 32 * pl.xts;
    pl.TXB = round_up(pl.TX + m - 1, 4);
    pl.TYB = sp::TY + m - 1;
    if (pl.TXB > 256 || pl.TYB > 256) return fail(ctx, DOCK_E_UNSUPPORTED, "sparse engine: TMA box too large");
    pl.ntx = (ctx->nx + pl.TX - 1) / pl.TX;
    pl.nty = (ctx->ny + sp::TY - 1) / sp::TY;
    pl.slot_words = round_up(pl.TXB * pl.TYB, 32);
    pl.box_bytes = pl.TXB * pl.TYB * 4;
    pl.GXp = round_up((pl.ntx - 1) * pl.TX + pl.TXB, 4);
    pl.GYp = (pl.nty - 1) * sp::TY + pl.TYB;
    pl.GZp = ctx->nz + m - 1;
    pl.ok = true;
    return DOCK_OK;
}

// Plane-ring depth for tmax atoms: as deep as shared memory allows (<= NPLMAX planes: the steps beyond the
// window m + PZ - 1 are TMA prefetch), at least the window; 0 when not even that fits.
int sp_npl(const SpPlan& pl, int m, int tmax, int zt)
{
    const int budget = kSmemLimit - 22 * 1024;   // static shared memory of k_corr_sparse: ~20 KB (lists, terms)
    for (int npl = sp::NPLMAX; npl >= m + sp::NPG * zt - 1; npl--)
        if ((size_t)std::max(tmax, 1) * npl * pl.slot_words * 4 <= (size_t)budget) return npl;
    return 0;
}

struct SpCall {   // one sparse-engine launch over the units of a call
    bool ok = false;
    int xts = 0;                      // translations per lane along x (row width 32 * xts)
    int zt = 1;                       // planes per warp and step
    int m = 0, tmax = 0, n_at = 0, atom_lo = 0, npl = 0, smem = 0;
    double terms = 0;                 // estimated occupied voxels summed over the units (cost model)
    std::vector<sp::Group> groups;    // rotation groups (<= sp::RB rotations of one probe)
};

// Host-side plan of a sparse-engine call: atom range of the probes the units touch, rotation groups,
// eligibility (atoms per probe <= sp::TMAX, plane ring fits shared memory).
dock_status sp_prepare(dock_ctx* ctx, int m, const dock_probe_desc* probes, int n_probes, int n_rot,
                       int64_t unit_begin, int64_t unit_end, SpCall* sc)
{
    sc->ok = false;
    sc->groups.clear();
    if (unit_end <= unit_begin) return DOCK_OK;
    const int p_lo = (int)(unit_begin / n_rot), p_hi = (int)((unit_end - 1) / n_rot);
    int atoms = 0, tmax = 0;
    std::vector<int> base(p_hi - p_lo + 1);
    for (int p = p_lo; p <= p_hi; p++) {
        base[p - p_lo] = atoms;
        atoms += probes[p].n_atoms;
        tmax = std::max(tmax, probes[p].n_atoms);
    }
    if (tmax > sp::TMAX) return DOCK_OK;
    // row width: the fewest wasted x translations whose plane ring fits shared memory for tmax atoms
    // (ties: 128, then 160, then 64 translations per row)
    int xts = 0, npl = 0, zt = 1, best_w = 1 << 30;
    for (int x : {4, 5, 2}) {
        if (make_sp_plan(ctx, m, x) != DOCK_OK) continue;
        // 64-translation rows: two planes per warp and step when the ring fits, else one
        int z = x == 2 ? 2 : 1, n = sp_npl(ctx->spplan[m][x], m, tmax, z);
        if (!n && z == 2) n = sp_npl(ctx->spplan[m][x], m, tmax, z = 1);
        const int w = (ctx->nx + 32 * x - 1) / (32 * x) * (32 * x);
        if (n && w < best_w) {
            best_w = w;
            xts = x;
            npl = n;
            zt = z;
        }
    }
    cudaGetLastError();
    ctx->err[0] = 0;
    if (!xts) return DOCK_OK;   // ineligible, not an error
    const SpPlan& pl = ctx->spplan[m][xts];
    sc->xts = xts;
    sc->zt = zt;
    int off = 0;
    for (int p = 0; p < p_lo; p++) off += probes[p].n_atoms;
    sc->m = m;
    sc->tmax = tmax;
    sc->n_at = atoms;
    sc->atom_lo = off;
    sc->npl = npl;
    sc->smem = std::max(tmax, 1) * npl * pl.slot_words * 4;
    sc->terms = 0;
    for (int p = p_lo; p <= p_hi; p++) {
        const int64_t u0 = std::max<int64_t>(unit_begin, (int64_t)p * n_rot);
        const int64_t u1 = std::min<int64_t>(unit_end, (int64_t)(p + 1) * n_rot);
        sc->terms += double(u1 - u0) * probes[p].n_atoms;
        for (int64_t u = u0; u < u1; u += sp::RB) {
            sp::Group gr;
            gr.slot0 = (int)(u - unit_begin);
            gr.n = (int)std::min<int64_t>(sp::RB, u1 - u);
            gr.atom0 = base[p - p_lo];
            gr.n_atoms = probes[p].n_atoms;
            sc->groups.push_back(gr);
        }
    }
    sc->ok = true;
    return DOCK_OK;
}

// Cost model of the engine choice (auto), per SM-clock rates measured on B200: the sparse
// engine gathers ~7.5 values (one per occupied voxel and translation); the tensor-core engine executes ~3000
// bf16 MACs (K-steps of 16 per rotation and translation, its bf16x3 split and padding included); the FFMA
// engine ~170 FP32 FMAs.
bool sp_better(dock_ctx* ctx, const SpCall& sc, int m, int n_units)
{
    if (!sc.ok) return false;
    const double ncell = (double)ctx->nx * ctx->ny * ctx->nz;
    const double sparse = sc.terms * ncell / 7.5;
    int v = 0, G = 0;
    double dense;
    if (plan_tc_launch(ctx, m, tc::ROT, &v, &G))
        dense = double(n_units) * ncell * ctx->tcplan[v][m].nsteps * 16.0 / 3000.0;
    else
        dense = double(n_units) * ncell * ctx->P * m * m * m / 170.0;
    return sparse < dense;
}

// Columns per item: minimise waves * (columns per item + per-item overhead, ~1 column: list warm-up and
// pipeline fill)
int sp_choose_cols(const dock_ctx* ctx, const SpPlan& pl, int64_t n_groups)
{
    const int ncol = pl.ntx * pl.nty;
    if (ctx->regions_override > 0) {   // DOCK_TUNE_REGIONS: regions (items) per rotation group
        const int G = std::min(ctx->regions_override, ncol);
        return (ncol + G - 1) / G;
    }
    int best = ncol;
    double best_cost = 1e300;
    for (int G = 1; G <= ncol; G++) {
        const int cpi = (ncol + G - 1) / G;
        const int geff = (ncol + cpi - 1) / cpi;
        const int64_t items = n_groups * geff;
        const int64_t waves = (items + ctx->n_sms - 1) / ctx->n_sms;
        const double cost = double(waves) * (cpi + 1.0);
        if (cost < best_cost - 1e-9) {
            best_cost = cost;
            best = cpi;
        }
    }
    return best;
}

// Per call: atom grids G_a of the touched probes (weights w) + their tensor map, and the occupied-voxel
// term tables of every unit.
dock_status sp_run_pre(dock_ctx* ctx, const SpCall& sc, int n_slots, int64_t unit_begin, int n_rot,
                       const double* d_xyz, const float* d_coef, const int* d_off, const double* d_rot, const float* w)
{
    const SpPlan& pl = ctx->spplan[sc.m][sc.xts];
    const size_t gcells = (size_t)pl.GXp * pl.GYp * pl.GZp;
    TRY(ensure(ctx, ctx->sp_G, sizeof(float) * gcells * std::max(sc.n_at, 1)));
    TRY(ensure(ctx, ctx->sp_tv, sizeof(int) * (size_t)n_slots * sp::TMAX));
    TRY(ensure(ctx, ctx->sp_ts, sizeof(int) * (size_t)n_slots * sp::TMAX));
    TRY(ensure(ctx, ctx->sp_nt, sizeof(int) * (size_t)n_slots));
    TRY(ensure(ctx, ctx->sp_dw, sizeof(float) * (size_t)n_slots * sp::TMAX * ctx->P));
    TRY(ensure(ctx, ctx->sp_slot_atoms, sizeof(int) * 2 * (size_t)n_slots));
    auto fn = encode_fn();
    if (!fn) return fail(ctx, DOCK_E_CUDA, "cuTensorMapEncodeTiled unavailable");
    cuuint64_t dims[4] = {(cuuint64_t)pl.GXp, (cuuint64_t)pl.GYp, (cuuint64_t)pl.GZp,
                          (cuuint64_t)std::max(sc.n_at, 1)};
    cuuint64_t strides[3] = {(cuuint64_t)pl.GXp * 4, (cuuint64_t)pl.GXp * pl.GYp * 4, (cuuint64_t)gcells * 4};
    cuuint32_t box[4] = {(cuuint32_t)pl.TXB, (cuuint32_t)pl.TYB, 1, 1};
    cuuint32_t es[4] = {1, 1, 1, 1};
    CUresult r = fn(&ctx->sp_tmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 4, ctx->sp_G.p, dims, strides, box, es,
                    CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                    CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (r != CUDA_SUCCESS) return fail(ctx, DOCK_E_CUDA, "cuTensorMapEncodeTiled (atom grids) failed (%d)", (int)r);
    if (sc.n_at > 0) {
        const size_t n4 = gcells / 4 * sc.n_at;
        const int blocks = (int)std::min<size_t>((n4 + 255) / 256, (size_t)ctx->n_sms * 16);
        sp::k_atom_grids<<<blocks, 256, 0, ctx->stream>>>(ctx->d_rec, ctx->geo.Xp, ctx->geo.Yp, ctx->geo.Zp, ctx->nx,
                                                         ctx->ny, ctx->nz, ctx->P, d_coef, w, sc.atom_lo, sc.n_at,
                                                         static_cast<float*>(ctx->sp_G.p), pl.GXp, pl.GYp, pl.GZp);
        CU(cudaGetLastError());
        ctx->kernels_last++;
    }
    sp::SpVoxArgs v{};
    v.xyz = d_xyz;
    v.coef = d_coef;
    v.atom_off = d_off;
    v.rot = d_rot;
    v.w = w;
    v.unit_begin = unit_begin;
    v.n_rot = n_rot;
    v.n_slots = n_slots;
    v.P = ctx->P;
    v.m = sc.m;
    v.spacing = ctx->spacing;
    v.term_v = static_cast<int*>(ctx->sp_tv.p);
    v.term_src = static_cast<int*>(ctx->sp_ts.p);
    v.n_terms = static_cast<int*>(ctx->sp_nt.p);
    v.dw = static_cast<float*>(ctx->sp_dw.p);
    v.status = ctx->d_small;
    v.slot_atoms = static_cast<int*>(ctx->sp_slot_atoms.p);
    v.atom_lo = sc.atom_lo;
    sp::k_voxelize_sparse<<<(n_slots + 127) / 128, 128, 0, ctx->stream>>>(v);
    CU(cudaGetLastError());
    ctx->kernels_last++;
    ctx->sp_natoms_last = sc.n_at;
    ctx->sp_tx_last = pl.TX;
    ctx->sp_zt_last = sc.zt;
    ctx->sp_terms_last = sc.terms;
    return DOCK_OK;
}

sp::SpArgs sp_args(dock_ctx* ctx, const SpCall& sc, const sp::Group* d_groups, int64_t n_groups)
{
    const SpPlan& pl = ctx->spplan[sc.m][sc.xts];
    sp::SpArgs a{};
    a.bound_every = ctx->sp_bound_every;
    a.nx = ctx->nx;
    a.ny = ctx->ny;
    a.nz = ctx->nz;
    a.m = sc.m;
    a.TX = pl.TX;
    a.ntx = pl.ntx;
    a.nty = pl.nty;
    a.TXB = pl.TXB;
    a.TYB = pl.TYB;
    a.slot_words = pl.slot_words;
    a.npl = sc.npl;
    a.cols_per_item = sp_choose_cols(ctx, pl, n_groups);
    a.G = (pl.ntx * pl.nty + a.cols_per_item - 1) / a.cols_per_item;
    a.box_bytes = pl.box_bytes;
    a.groups = d_groups;
    a.term_v = static_cast<const int*>(ctx->sp_tv.p);
    a.term_src = static_cast<const int*>(ctx->sp_ts.p);
    a.n_terms = static_cast<const int*>(ctx->sp_nt.p);
    a.dw = static_cast<const float*>(ctx->sp_dw.p);
    a.P = ctx->P;
    a.rec = ctx->d_rec;
    a.rXp = ctx->geo.Xp;
    a.rYp = ctx->geo.Yp;
    a.rZp = ctx->geo.Zp;
    return a;
}

// Pack folded FP32 weights into the tcgen05 A-operand layout of variant v.  Variant 1 first builds the
// occupancy schedule (dock_tc.cuh): unit K-step masks and the greedy block clustering (main pass, m <= 4,
// DOCK_TUNE_TC_SCHEDULE 0), then per block the table of occupied K-steps, then the A operand in table order.
// fb: the fallback's buffers (no clustering; n_live = the live count of the device-driven loop).
dock_status pack_weights_tc(dock_ctx* ctx, int m, int v, int n_slots, const float* Lw, bool fb = false,
                            const unsigned* n_live = nullptr, bool shard = false)
{
    const TcPlan& tp = ctx->tcplan[v][m];
    const int64_t n_blocks = (n_slots + tc::ROT - 1) / tc::ROT;
    DevBuf& Wb = fb ? ctx->fb_W : ctx->Wtc;
    TRY(ensure(ctx, Wb, (size_t)n_blocks * tp.nsteps * tc::WCHUNK));
    const int64_t rows = n_blocks * tp.nsteps * 2 * tc::ROT;
    const int grid = (int)std::min<int64_t>((rows + 255) / 256, 65535);
    unsigned char* W = static_cast<unsigned char*>(Wb.p);
    if (v == 1) {
        DevBuf& ks = fb ? ctx->fb_ksrc : ctx->tc_ksrc;
        DevBuf& ki = fb ? ctx->fb_kinfo : ctx->tc_kinfo;
        TRY(ensure(ctx, ks, sizeof(uint16_t) * n_blocks * tp.nsteps));
        TRY(ensure(ctx, ki, sizeof(int4) * n_blocks));
        const int* perm = nullptr;
        const int nstg = tp.nsteps / tc::KSTEPS;
        const bool masked = ctx->tc_sched != 2 && nstg <= 64;
        const unsigned long long* um = nullptr;
        if (masked) {   // per-unit stage masks (positions past the live count: none)
            TRY(ensure(ctx, fb ? ctx->fb_umask : ctx->tc_umask, sizeof(unsigned long long) * n_slots));
            auto* umw = static_cast<unsigned long long*>((fb ? ctx->fb_umask : ctx->tc_umask).p);
            const int warps = (n_slots + dk::RB - 1) / dk::RB;
            tc::k_tc_unit_masks<<<(warps + 3) / 4, 128, 0, ctx->stream>>>(Lw, n_slots, n_live, ctx->P, m, umw);
            CU(cudaGetLastError());
            ctx->kernels_last++;
            um = umw;
        }
        if (masked && !fb && ctx->tc_sched == 0 && n_slots > tc::ROT) {
            TRY(ensure(ctx, ctx->tc_perm, sizeof(int) * n_blocks * tc::ROT));
            const int windows = (n_slots + tc::CL_W - 1) / tc::CL_W;
            if (nstg <= tc::CB_BITS) {   // distinct masks fit a histogram
                TRY(ensure(ctx, ctx->tc_sorted, sizeof(int) * n_slots));
                const int sm = (int)sizeof(tc::ClusterBinsSmem);
                CU(cudaFuncSetAttribute(tc::k_tc_cluster_bins, cudaFuncAttributeMaxDynamicSharedMemorySize, sm));
                tc::k_tc_cluster_bins<<<windows, tc::CL_THREADS, sm, ctx->stream>>>(
                    um, n_slots, static_cast<int*>(ctx->tc_sorted.p), static_cast<int*>(ctx->tc_perm.p));
            } else {
                tc::k_tc_cluster<<<windows, tc::CL_THREADS, 0, ctx->stream>>>(um, n_slots,
                                                                               static_cast<int*>(ctx->tc_perm.p));
            }
            CU(cudaGetLastError());
            ctx->kernels_last++;
            perm = static_cast<const int*>(ctx->tc_perm.p);
        }
        if (!fb) {
            ctx->tc_perm_on = perm != nullptr;
            ctx->tc_nblk_local = -1;
            if (shard && ctx->shard_world > 1) {   // block sharding: this rank's blocks of the (clustered) block order
                TRY(ensure(ctx, ctx->tc_blkmap, sizeof(int) * n_blocks));
                TRY(ensure(ctx, ctx->tc_owned, (size_t)n_slots));
                tc::k_tc_shard_blocks<<<(int)std::min<int64_t>((n_blocks * tc::ROT + 255) / 256, 4096), 256, 0,
                                        ctx->stream>>>(perm, n_slots, (int)n_blocks, ctx->shard_rank, ctx->shard_world,
                                                       static_cast<int*>(ctx->tc_blkmap.p),
                                                       static_cast<unsigned char*>(ctx->tc_owned.p));
                CU(cudaGetLastError());
                ctx->kernels_last++;
                ctx->tc_nblk_local =
                    n_blocks > ctx->shard_rank ? (int)((n_blocks - ctx->shard_rank + ctx->shard_world - 1) / ctx->shard_world) : 0;
            }
        }
        tc::k_tc_block_tables<<<(int)n_blocks, 128, 0, ctx->stream>>>(
            um, perm, n_slots, tp.nsteps, static_cast<uint16_t*>(ks.p), static_cast<int4*>(ki.p),
            fb ? nullptr : reinterpret_cast<unsigned*>(ctx->d_small + 3));
        CU(cudaGetLastError());
        tc::k_pack_weights_tc1<<<grid, 256, 0, ctx->stream>>>(Lw, perm, static_cast<const uint16_t*>(ks.p),
                                                               static_cast<const int4*>(ki.p), W, n_slots, ctx->P,
                                                               m, tp.nsteps);
        ctx->kernels_last++;
        if (!fb) ctx->tc_blocks_last = (int)n_blocks;
    } else {
        tc::k_pack_weights_tcs<<<grid, 256, 0, ctx->stream>>>(Lw, W, n_slots, ctx->P, m, tp.nsteps);
    }
    CU(cudaGetLastError());
    ctx->kernels_last++;
    return DOCK_OK;
}

// FFT engine (engine 3): score grids of n slots [slot0, slot0 + n) (dock_fft.h).
dock_status run_grid_fft(dock_ctx* ctx, int m, int slot0, int n, const float* Lw, float* grid)
{
    if (!ctx->fft && !(ctx->fft = dock_fft_create())) return fail(ctx, DOCK_E_OOM, "FFT engine state");
    const dk::Geo& G = ctx->geo;
    cudaError_t e = dock_fft_grids(ctx->fft, ctx->d_rec, G.Xp, G.Yp, G.Zp, ctx->nx, ctx->ny, ctx->nz, ctx->P, m, Lw,
                                   slot0, n, grid, ctx->stream);
    if (e != cudaSuccess) return fail(ctx, DOCK_E_CUDA, "FFT engine: %s", cudaGetErrorString(e));
    ctx->kernels_last += 5;   // memset, scatter, R2C, multiply-accumulate, C2R
    return DOCK_OK;
}

// FFT engine poses: score grids in chunks, then the exact greedy of the fallback path.
dock_status run_fft_poses(dock_ctx* ctx, int m, int n_units, int64_t unit_begin, int n_rot, int k, int rho,
                          void* poses)
{
    const int chunk = std::min(n_units, dock_fft_batch(ctx->nx, ctx->ny, ctx->nz, ctx->P));
    const size_t ncell = (size_t)ctx->nx * ctx->ny * ctx->nz;
    TRY(ensure(ctx, ctx->grid, sizeof(float) * ncell * chunk));
    TRY(ensure(ctx, ctx->slots, sizeof(int) * n_units));
    TRY(ensure(ctx, ctx->picks, sizeof(unsigned long long) * chunk * k));
    TRY(ensure_pinned(ctx, sizeof(int) * n_units));
    int* h = static_cast<int*>(ctx->h_stage);
    CU(cudaStreamSynchronize(ctx->stream));
    for (int i = 0; i < n_units; i++) h[i] = i;   // output slot of grid i
    CU(cudaMemcpyAsync(ctx->slots.p, h, sizeof(int) * n_units, cudaMemcpyHostToDevice, ctx->stream));
    for (int c0 = 0; c0 < n_units; c0 += chunk) {
        const int n = std::min(chunk, n_units - c0);
        TRY(run_grid_fft(ctx, m, c0, n, static_cast<const float*>(ctx->Lw.p), static_cast<float*>(ctx->grid.p)));
        dk::GreedyArgs ga{};
        ga.grid = static_cast<const float*>(ctx->grid.p);
        ga.slots = static_cast<const int*>(ctx->slots.p) + c0;
        ga.picks = static_cast<unsigned long long*>(ctx->picks.p);
        ga.n = n;
        ga.k = k;
        ga.rho = rho;
        ga.n_rot = n_rot;
        ga.nx = ctx->nx;
        ga.ny = ctx->ny;
        ga.nz = ctx->nz;
        ga.unit_begin = unit_begin;
        ga.poses = poses;
        ga.flag_bits = 0u;
        dk::k_fill_u64<<<1, 256, 0, ctx->stream>>>(ga.picks, (size_t)n * k, dk::KEY_MAX);
        CU(cudaGetLastError());
        const int per_grid = std::max(8, std::min(512, 16 * ctx->n_sms / std::max(1, n)));
        for (int j = 0; j < k; j++) {
            ga.round = j;
            dk::k_greedy_round<<<n * per_grid, 256, 0, ctx->stream>>>(ga);
            CU(cudaGetLastError());
        }
        dk::k_greedy_emit<<<(n * k + 127) / 128, 128, 0, ctx->stream>>>(ga);
        CU(cudaGetLastError());
        ctx->kernels_last += k + 2;
    }
    return DOCK_OK;
}

// Score grids for n slots with the tensor-core engine (GRID epilogue).
dock_status run_grid_tc(dock_ctx* ctx, int m, int n_slots, const float* Lw, float* grid)
{
    const int64_t n_blocks = (n_slots + tc::ROT - 1) / tc::ROT;
    int v = 0, G = 0;
    if (!plan_tc_launch(ctx, m, n_slots, &v, &G)) return fail(ctx, DOCK_E_UNSUPPORTED, "no tensor-core plan");
    TRY(pack_weights_tc(ctx, m, v, n_slots, Lw));
    tc::TcArgs a = tc_args(ctx, m, v, n_slots, G, static_cast<const unsigned char*>(ctx->Wtc.p));
    a.grid = grid;
    const int64_t items = tc_ctas(a, n_slots, ctx->n_sms);
    if (items > 0x7fffffff || n_blocks > 0x7fffffff) return fail(ctx, DOCK_E_UNSUPPORTED, "too many work items");
    CU(launch_tc(m, v, true, ctx->tcplan[v][m], a, (int)items, ctx->stream));
    ctx->kernels_last++;
    return DOCK_OK;
}

// ---------------------------------------------------------------- device-driven exact fallback
//
// Rotations k_merge flagged (candidate overflow, or a list whose last key is below the last pick; DESIGN.md
// §8) get their full score grid from the engine that produced their candidates (tcgen05 GRID epilogue or
// FFMA GRID epilogue: identical score bits) and the exact best-then-exclude greedy.  The
// number of flagged rotations is only known on the device, so the fallback is one CUDA graph:
//   k_fb_init (condition = fb_cnt > 0) -> WHILE { k_fb_chunk -> k_voxelize_dyn -> [pack] -> GRID correlation
//   -> k_fill_u64 -> k rounds k_greedy_round -> k_greedy_emit -> k_fb_advance (condition = more left) }
// over chunks of `ch` flagged slots.  Every per-call value (poses, unit_begin, n_rot, input pointers) is
// read from the dk::FbDyn block uploaded with the call's inputs, so the instantiated graph is reused
// across calls with the same shape; the host never waits for the flag count.

struct FbKey {   // everything the captured fallback graph bakes in (compared bytewise)
    int m, kind, v, G, k, rho, ch, nepi, P, nx, ny, nz;
    int sp_nat, sp_npl, sp_smem, sp_xts;
    const void *fb_list, *d_small, *dyn, *grid, *Lw, *W, *picks, *slots, *ctl, *w, *ksrc, *kinfo, *umask;
    const void *spG, *sp_tv, *sp_ts, *sp_nt, *sp_dw, *sp_sa, *fb_groups;
};
static_assert(sizeof(FbKey) <= sizeof(((dock_ctx*)nullptr)->fb_key), "fb_key too small");

int fb_chunk(const dock_ctx* ctx, int kind)
{
    const bool use_tc = kind == ENG_TC;
    const size_t ncell = (size_t)ctx->nx * ctx->ny * ctx->nz;
    const size_t budget = size_t(1) << 30;   // score grids of one chunk: <= 1 GiB
    const size_t fit = std::max<size_t>(1, budget / (ncell * sizeof(float)));
    return (int)std::min<size_t>(use_tc ? tc::ROT : 64, fit);
}

dock_status fb_buffers(dock_ctx* ctx, int m, int ch, int k)
{
    const size_t ncell = (size_t)ctx->nx * ctx->ny * ctx->nz;
    const int m3 = m * m * m;
    TRY(ensure(ctx, ctx->fb_grid, sizeof(float) * ncell * ch));
    TRY(ensure(ctx, ctx->fb_Lw, sizeof(float) * ((ch + dk::RB - 1) / dk::RB) * dk::RB * ctx->P * m3));
    TRY(ensure(ctx, ctx->fb_picks, sizeof(unsigned long long) * ch * k));
    TRY(ensure(ctx, ctx->fb_slots, sizeof(int) * ch));
    TRY(ensure(ctx, ctx->fb_ctl, sizeof(dk::FbCtl)));
    TRY(ensure(ctx, ctx->fb_groups, sizeof(sp::Group) * ch));
    return DOCK_OK;
}

// Capture + instantiate the fallback graph for this key (ctx->stream is redirected to the private capture
// streams while the existing launch helpers record into the graph).
// One iteration of the fallback loop on stream st (the kernels read the chunk from the device-side control
// block): chunk -> [voxelize] -> GRID correlation -> greedy rounds -> emit.  Captured into the WHILE body of
// the fallback graph, or launched from a host loop (DOCK_FB_HOST_LOOP=1: sanitizer runs, whose tools do not
// support conditional graph nodes).
dock_status enqueue_fb_body(dock_ctx* ctx, const FbKey& key, const dk::FbDyn* d_dyn, const SpCall* sc, cudaStream_t st)
{
    const int m = key.m, ch = key.ch, k = key.k;
    auto* fb_cnt = reinterpret_cast<unsigned int*>(ctx->d_small + 1);
    auto* ctl = static_cast<dk::FbCtl*>(ctx->fb_ctl.p);
    int* slots = static_cast<int*>(ctx->fb_slots.p);
    cudaStream_t user = ctx->stream;
    ctx->stream = st;   // the launch helpers below enqueue on ctx->stream
    auto body = [&]() -> dock_status {
        dk::k_fb_chunk<<<1, 128, 0, st>>>(fb_cnt, static_cast<const int*>(ctx->fb_list.p), ctl, slots, ch);
        CU(cudaGetLastError());
        const float* Lw = static_cast<const float*>(ctx->fb_Lw.p);
        float* grid = static_cast<float*>(ctx->fb_grid.p);
        if (key.kind == ENG_SPARSE) {
            // the main pass's atom grids and term tables stay valid until the next call: one single-rotation
            // group per flagged slot, GRID epilogue into row = chunk position
            auto* groups = static_cast<sp::Group*>(ctx->fb_groups.p);
            sp::k_sparse_fb_groups<<<(ch + 127) / 128, 128, 0, st>>>(
                slots, &ctl->n_live, static_cast<const int*>(ctx->sp_slot_atoms.p), groups, ch);
            CU(cudaGetLastError());
            sp::SpArgs a = sp_args(ctx, *sc, groups, ch);
            a.grid = grid;
            a.n_live = &ctl->n_live;
            CU(dock_launch_sparse(sc->xts, sc->zt, true, ctx->sp_tmap, sc->smem, a, (int)(ch * a.G), st));
        } else {
            const int nvox = (ch + dk::RB - 1) / dk::RB * dk::RB * ctx->P;
            dk::k_voxelize_dyn<<<(nvox + 127) / 128, 128, 0, st>>>(&d_dyn->vox);
            CU(cudaGetLastError());
            if (key.kind == ENG_TC) {
                TRY(pack_weights_tc(ctx, m, key.v, ch, Lw, true, &ctl->n_live));
                tc::TcArgs a = tc_args(ctx, m, key.v, ch, key.G, static_cast<const unsigned char*>(ctx->fb_W.p));
                a.grid = grid;
                a.n_live = &ctl->n_live;
                a.trace = nullptr;
                CU(launch_tc(m, key.v, true, ctx->tcplan[key.v][m], a, (int)tc_ctas(a, ch, ctx->n_sms), st));
            } else {
                const int64_t nb = (ch + dk::RB - 1) / dk::RB;
                dk::CorrArgs a = corr_args(ctx, m, ch, key.G, Lw);
                a.grid = grid;
                a.n_live = &ctl->n_live;
                CU(dock_launch_ffma(m, true, ctx->plan[m].tmap, ctx->plan[m].smem, a, (int)(nb * key.G), st));
            }
        }
        dk::GreedyArgs ga{};
        ga.grid = grid;
        ga.slots = slots;
        ga.picks = static_cast<unsigned long long*>(ctx->fb_picks.p);
        ga.n = ch;
        ga.k = k;
        ga.rho = key.rho;
        ga.nx = ctx->nx;
        ga.ny = ctx->ny;
        ga.nz = ctx->nz;
        ga.flag_bits = 1u;   // DOCK_POSE_FALLBACK
        ga.n_live = &ctl->n_live;
        ga.dyn = d_dyn;
        dk::k_fill_u64<<<1, 256, 0, st>>>(ga.picks, (size_t)ch * k, dk::KEY_MAX);
        CU(cudaGetLastError());
        const int per_grid = std::max(8, std::min(512, 16 * ctx->n_sms / std::max(1, ch)));
        for (int j = 0; j < k; j++) {
            ga.round = j;
            dk::k_greedy_round<<<ch * per_grid, 256, 0, st>>>(ga);
            CU(cudaGetLastError());
        }
        dk::k_greedy_emit<<<(ch * k + 127) / 128, 128, 0, st>>>(ga);
        CU(cudaGetLastError());
        return DOCK_OK;
    };
    const dock_status r = body();
    ctx->stream = user;
    return r;
}

dock_status build_fb_graph(dock_ctx* ctx, const FbKey& key, const dk::FbDyn* d_dyn, const SpCall* sc)
{
    if (ctx->fb_exec) {
        cudaGraphExecDestroy(ctx->fb_exec);
        ctx->fb_exec = nullptr;
    }
    auto* fb_cnt = reinterpret_cast<unsigned int*>(ctx->d_small + 1);
    auto* ctl = static_cast<dk::FbCtl*>(ctx->fb_ctl.p);
    cudaStream_t cs = ctx->cap_stream, cs2 = ctx->cap_stream2;
    cudaGraph_t graph = nullptr;
    auto body = [&]() -> dock_status {
        CU(cudaStreamBeginCapture(cs, cudaStreamCaptureModeThreadLocal));
        cudaStreamCaptureStatus cst;
        cudaGraph_t g = nullptr;
        const cudaGraphNode_t* deps = nullptr;
        size_t nd = 0;
        CU(cudaStreamGetCaptureInfo(cs, &cst, nullptr, &g, &deps, &nd));
        cudaGraphConditionalHandle h;
        CU(cudaGraphConditionalHandleCreate(&h, g, 0, 0));
        dk::k_fb_init<<<1, 1, 0, cs>>>(h, fb_cnt, ctl);
        CU(cudaGetLastError());
        CU(cudaStreamGetCaptureInfo(cs, &cst, nullptr, &g, &deps, &nd));
        cudaGraphNodeParams cp = {};
        cp.type = cudaGraphNodeTypeConditional;
        cp.conditional.handle = h;
        cp.conditional.type = cudaGraphCondTypeWhile;
        cp.conditional.size = 1;
        cudaGraphNode_t node;
        CU(cudaGraphAddNode(&node, g, deps, nd, &cp));
        cudaGraph_t loop = cp.conditional.phGraph_out[0];
        CU(cudaStreamUpdateCaptureDependencies(cs, &node, 1, cudaStreamSetCaptureDependencies));
        // loop body, captured on the second private stream
        CU(cudaStreamBeginCaptureToGraph(cs2, loop, nullptr, nullptr, 0, cudaStreamCaptureModeThreadLocal));
        TRY(enqueue_fb_body(ctx, key, d_dyn, sc, cs2));
        dk::k_fb_advance<<<1, 1, 0, cs2>>>(h, fb_cnt, ctl, key.ch);
        CU(cudaGetLastError());
        CU(cudaStreamEndCapture(cs2, nullptr));
        CU(cudaStreamEndCapture(cs, &graph));
        CU(cudaGraphInstantiate(&ctx->fb_exec, graph, 0));
        return DOCK_OK;
    };
    const dock_status st = body();
    if (st != DOCK_OK) {   // leave no capture open on the private streams
        cudaGraph_t junk = nullptr;
        cudaStreamCaptureStatus cst;
        if (cudaStreamIsCapturing(cs2, &cst) == cudaSuccess && cst != cudaStreamCaptureStatusNone)
            cudaStreamEndCapture(cs2, &junk);
        if (cudaStreamIsCapturing(cs, &cst) == cudaSuccess && cst != cudaStreamCaptureStatusNone)
            cudaStreamEndCapture(cs, &junk);
        if (junk) cudaGraphDestroy(junk);
        cudaGetLastError();
        memset(ctx->fb_key, 0, sizeof(ctx->fb_key));
    }
    if (graph) cudaGraphDestroy(graph);
    return st;
}

// Enqueue the fallback graph on the context stream (no host synchronisation).
dock_status launch_fallback(dock_ctx* ctx, int m, int kind, int k, int rho, const dk::FbDyn* d_dyn,
                            const SpCall* sc)
{
    const int ch = fb_chunk(ctx, kind);
    TRY(fb_buffers(ctx, m, ch, k));
    FbKey key;
    memset(&key, 0, sizeof(key));
    key.m = m;
    key.kind = kind;
    if (kind == ENG_SPARSE) {
        key.sp_nat = sc->n_at;
        key.sp_npl = sc->npl;
        key.sp_smem = sc->smem;
        key.sp_xts = sc->xts * 8 + sc->zt;
        key.spG = ctx->sp_G.p;
        key.sp_tv = ctx->sp_tv.p;
        key.sp_ts = ctx->sp_ts.p;
        key.sp_nt = ctx->sp_nt.p;
        key.sp_dw = ctx->sp_dw.p;
        key.sp_sa = ctx->sp_slot_atoms.p;
        key.fb_groups = ctx->fb_groups.p;
    } else if (kind == ENG_TC) {
        int vv = 0, G = 0;
        if (!plan_tc_launch(ctx, m, ch, &vv, &G)) return fail(ctx, DOCK_E_UNSUPPORTED, "no tensor-core plan");
        key.v = vv;
        key.G = G;
        const TcPlan& tp = ctx->tcplan[vv][m];
        TRY(ensure(ctx, ctx->fb_W, (size_t)tp.nsteps * tc::WCHUNK));
        TRY(ensure(ctx, ctx->fb_ksrc, sizeof(uint16_t) * tp.nsteps));
        TRY(ensure(ctx, ctx->fb_umask, sizeof(unsigned long long) * ch));
        TRY(ensure(ctx, ctx->fb_kinfo, sizeof(int4)));
    } else if (kind == ENG_FFMA) {
        key.G = choose_regions(ctx, (ch + dk::RB - 1) / dk::RB);
    }
    key.k = k;
    key.rho = rho;
    key.ch = ch;
    key.nepi = ctx->tc_nepi;
    key.P = ctx->P;
    key.nx = ctx->nx;
    key.ny = ctx->ny;
    key.nz = ctx->nz;
    key.fb_list = ctx->fb_list.p;
    key.d_small = ctx->d_small;
    key.dyn = d_dyn;
    key.grid = ctx->fb_grid.p;
    key.Lw = ctx->fb_Lw.p;
    key.W = ctx->fb_W.p;
    key.ksrc = ctx->fb_ksrc.p;
    key.kinfo = ctx->fb_kinfo.p;
    key.umask = ctx->fb_umask.p;
    key.picks = ctx->fb_picks.p;
    key.slots = ctx->fb_slots.p;
    key.ctl = ctx->fb_ctl.p;
    key.w = ctx->d_w;
    if (ctx->fb_host_loop) {   // diagnostic mode: the same kernels from a host loop (synchronises)
        auto* ctl = static_cast<dk::FbCtl*>(ctx->fb_ctl.p);
        CU(cudaMemcpyAsync(ctx->h_small, ctx->d_small, 16, cudaMemcpyDeviceToHost, ctx->stream));
        CU(cudaStreamSynchronize(ctx->stream));
        const int n = ctx->h_small[1];
        dk::k_fb_init_plain<<<1, 1, 0, ctx->stream>>>(ctl);
        CU(cudaGetLastError());
        for (int done = 0; done < n; done += ch) {
            TRY(enqueue_fb_body(ctx, key, d_dyn, sc, ctx->stream));
            dk::k_fb_advance_plain<<<1, 1, 0, ctx->stream>>>(ctl, ch);
            CU(cudaGetLastError());
        }
        return DOCK_OK;
    }
    if (!ctx->fb_exec || memcmp(&key, ctx->fb_key, sizeof(key)) != 0) {
        TRY(build_fb_graph(ctx, key, d_dyn, sc));
        memcpy(ctx->fb_key, &key, sizeof(key));
    }
    CU(cudaGraphLaunch(ctx->fb_exec, ctx->stream));
    ctx->kernels_last++;   // k_fb_init; the loop body runs only for flagged rotations
    return DOCK_OK;
}

// Template of the per-call fallback arguments (the input pointers are filled by stage_inputs).
dk::FbDyn fb_template(dock_ctx* ctx, int m, int ch, int64_t unit_begin, int n_rot, void* poses)
{
    dk::FbDyn f;
    memset(&f, 0, sizeof(f));
    f.vox.w = ctx->d_w;
    f.vox.unit_list = static_cast<const int*>(ctx->fb_slots.p);
    f.vox.unit_begin = unit_begin;
    f.vox.n_rot = n_rot;
    f.vox.n_slots = ch;
    f.vox.P = ctx->P;
    f.vox.m = m;
    f.vox.spacing = ctx->spacing;
    f.vox.Lw = static_cast<float*>(ctx->fb_Lw.p);
    f.vox.status = ctx->d_small;
    f.vox.n_live = &static_cast<dk::FbCtl*>(ctx->fb_ctl.p)->n_live;
    f.poses = poses;
    f.unit_begin = unit_begin;
    f.n_rot = n_rot;
    return f;
}

// Queue the copy of the status words for the next sync point (asynchronous).
dock_status end_call(dock_ctx* ctx)
{
    CU(cudaMemcpyAsync(ctx->h_small, ctx->d_small, 16, cudaMemcpyDeviceToHost, ctx->stream));
    CU(cudaEventRecord(ctx->ev_done, ctx->stream));
    ctx->unsynced = true;
    return DOCK_OK;
}

// Sync point: wait for the context stream, take the stats of the last call and report (then clear) the
// sticky device status bits of every call since the previous sync point.
dock_status sync_point(dock_ctx* ctx)
{
    CU(cudaStreamSynchronize(ctx->stream));
    ctx->unsynced = false;
    ctx->fallback_last = (unsigned)ctx->h_small[1];
    ctx->cand_max_last = (unsigned)ctx->h_small[2];
    const int st = ctx->h_small[0];
    if (st) {
        ctx->h_small[0] = 0;
        CU(cudaMemsetAsync(ctx->d_small, 0, 4, ctx->stream));
        CU(cudaStreamSynchronize(ctx->stream));
        if (st & dk::ST_BAD_ROTATION)
            return fail(ctx, DOCK_E_BAD_ROTATION, "a rotation is not a proper rotation matrix");
        if (st & dk::ST_OUTSIDE)
            return fail(ctx, DOCK_E_PROBE_OUTSIDE_GRID, "a probe atom voxelizes outside the m^3 probe box");
    }
    return DOCK_OK;
}

}  // namespace

// =====================================================================================  ABI

extern "C" {

const char* dock_status_string(dock_status s)
{
    switch (s) {
        case DOCK_OK: return "DOCK_OK";
        case DOCK_E_INVALID_ARG: return "DOCK_E_INVALID_ARG";
        case DOCK_E_UNSUPPORTED: return "DOCK_E_UNSUPPORTED";
        case DOCK_E_PROBE_OUTSIDE_GRID: return "DOCK_E_PROBE_OUTSIDE_GRID";
        case DOCK_E_BAD_ROTATION: return "DOCK_E_BAD_ROTATION";
        case DOCK_E_CUDA: return "DOCK_E_CUDA";
        case DOCK_E_OOM: return "DOCK_E_OOM";
    }
    return "DOCK_E_UNKNOWN";
}

const char* dock_last_error(const dock_ctx* ctx) { return ctx ? ctx->err : "null context"; }

void dock_destroy(dock_ctx* ctx)
{
    if (!ctx) return;
    cudaSetDevice(ctx->device);
    if (ctx->stream) cudaStreamSynchronize(ctx->stream);
    DevBuf* bufs[] = {&ctx->xyz,     &ctx->coef,     &ctx->off,    &ctx->rot,      &ctx->Lw,       &ctx->T,
                      &ctx->mu,      &ctx->cnt,      &ctx->cand,   &ctx->poses,    &ctx->fb_list,  &ctx->grid,
                      &ctx->slots,   &ctx->units,    &ctx->Lw_fb,  &ctx->picks,    &ctx->fb_grid,  &ctx->fb_Lw,
                      &ctx->fb_W,    &ctx->fb_picks, &ctx->fb_slots, &ctx->fb_ctl,   &ctx->tc_ksrc,
                      &ctx->tc_kinfo, &ctx->tc_perm, &ctx->tc_umask, &ctx->tc_sorted, &ctx->fb_ksrc, &ctx->fb_kinfo,
                      &ctx->fb_umask, &ctx->tc_seg,  &ctx->tc_pref, &ctx->tc_blkmap, &ctx->tc_owned};
    for (DevBuf* b : bufs)
        if (b->p) cudaFree(b->p);
    if (ctx->d_trace) cudaFree(ctx->d_trace);
    if (ctx->d_sched) cudaFree(ctx->d_sched);
    if (ctx->fft) dock_fft_destroy(ctx->fft);
    if (ctx->d_rec) cudaFree(ctx->d_rec);
    if (ctx->d_rec_tc) cudaFree(ctx->d_rec_tc);
    if (ctx->d_rec_pair) cudaFree(ctx->d_rec_pair);
    if (ctx->Wtc.p) cudaFree(ctx->Wtc.p);
    if (ctx->d_w) cudaFree(ctx->d_w);
    if (ctx->d_eye) cudaFree(ctx->d_eye);
    if (ctx->d_ones) cudaFree(ctx->d_ones);
    if (ctx->d_small) cudaFree(ctx->d_small);
    if (ctx->h_small) cudaFreeHost(ctx->h_small);
    if (ctx->h_stage) cudaFreeHost(ctx->h_stage);
    for (auto& st : ctx->stage) {
        if (st.h) cudaFreeHost(st.h);
        if (st.ev) cudaEventDestroy(st.ev);
    }
    if (ctx->fb_exec) cudaGraphExecDestroy(ctx->fb_exec);
    if (ctx->ev_done) cudaEventDestroy(ctx->ev_done);
    if (ctx->cap_stream) cudaStreamDestroy(ctx->cap_stream);
    if (ctx->cap_stream2) cudaStreamDestroy(ctx->cap_stream2);
    for (cudaEvent_t e : ctx->ev_corr)
        if (e) cudaEventDestroy(e);
    if (ctx->own_stream && ctx->stream) cudaStreamDestroy(ctx->stream);
    cudaGetLastError();
    delete ctx;
}

dock_status dock_init(const dock_grid_desc* g, const float* receptor, const float* weights, dock_ctx** out)
{
    if (!out) return DOCK_E_INVALID_ARG;
    *out = nullptr;
    if (!g || !receptor || !weights) return DOCK_E_INVALID_ARG;
    if (g->nx < 1 || g->ny < 1 || g->nz < 1 || g->n_terms < 1 || g->m_max < 1 || !(g->spacing > 0.0) ||
        !std::isfinite(g->spacing))
        return DOCK_E_INVALID_ARG;
    if (g->n_terms > DOCK_MAX_TERMS || g->m_max > DOCK_MAX_M) return DOCK_E_UNSUPPORTED;
    if ((int64_t)g->nx * g->ny * g->nz >= (int64_t(1) << 31) - 1) return DOCK_E_UNSUPPORTED;

    dock_ctx* ctx = new (std::nothrow) dock_ctx();
    if (!ctx) return DOCK_E_OOM;
    ctx->device = g->device;
    ctx->nx = g->nx;
    ctx->ny = g->ny;
    ctx->nz = g->nz;
    ctx->P = g->n_terms;
    ctx->m_max = g->m_max;
    ctx->spacing = g->spacing;
    auto bail = [&](dock_status s) {
        dock_destroy(ctx);
        return s;
    };
    if (cudaSetDevice(ctx->device) != cudaSuccess) {
        cudaGetLastError();
        return bail(DOCK_E_CUDA);
    }
    if (g->stream) {
        ctx->stream = static_cast<cudaStream_t>(g->stream);
    } else {
        if (cudaStreamCreateWithFlags(&ctx->stream, cudaStreamNonBlocking) != cudaSuccess) return bail(DOCK_E_CUDA);
        ctx->own_stream = true;
    }
    if (cudaEventCreate(&ctx->ev_corr[0]) != cudaSuccess || cudaEventCreate(&ctx->ev_corr[1]) != cudaSuccess ||
        cudaEventCreateWithFlags(&ctx->ev_done, cudaEventDisableTiming) != cudaSuccess ||
        cudaStreamCreateWithFlags(&ctx->cap_stream, cudaStreamNonBlocking) != cudaSuccess ||
        cudaStreamCreateWithFlags(&ctx->cap_stream2, cudaStreamNonBlocking) != cudaSuccess)
        return bail(DOCK_E_CUDA);
    for (auto& st : ctx->stage)
        if (cudaEventCreateWithFlags(&st.ev, cudaEventDisableTiming) != cudaSuccess) return bail(DOCK_E_CUDA);
    if (const char* e = getenv("DOCK_FB_HOST_LOOP")) ctx->fb_host_loop = atoi(e);
    if (const char* e = getenv("DOCK_TC_SEG_COST")) ctx->tc_seg_cost = std::max(0, atoi(e));   // tuning experiments
    if (const char* e = getenv("DOCK_SP_BOUND_EVERY")) ctx->sp_bound_every = std::max(0, atoi(e));
    if (const char* e = getenv("DOCK_TC_TRACE")) {
        if (atoi(e) > 0 && cudaMalloc(&ctx->d_trace, sizeof(unsigned long long) * tc::TR_N) != cudaSuccess)
            return bail(DOCK_E_OOM);
    }
    int v = 0;
    if (cudaDeviceGetAttribute(&v, cudaDevAttrMultiProcessorCount, ctx->device) == cudaSuccess) ctx->n_sms = v;
    if (cudaDeviceGetAttribute(&v, cudaDevAttrL2CacheSize, ctx->device) == cudaSuccess) ctx->l2_bytes = v;
    ctx->geo = choose_geo(ctx->nx, ctx->ny, ctx->nz, ctx->m_max);
    const dk::Geo& G = ctx->geo;
    const int P = ctx->P;
    const size_t n_in = (size_t)P * ctx->nx * ctx->ny * ctx->nz;
    const size_t n_pad = (size_t)P * G.Xp * G.Yp * G.Zp;

    // weights (host or device) -> host copy for validation
    std::vector<float> w(P);
    const int wk = ptr_kind(weights, ctx->device), rk = ptr_kind(receptor, ctx->device);
    if (wk < 0 || rk < 0) return bail(DOCK_E_INVALID_ARG);   // device memory of another device
    if (wk == 1) {
        if (cudaMemcpy(w.data(), weights, sizeof(float) * P, cudaMemcpyDeviceToHost) != cudaSuccess)
            return bail(DOCK_E_CUDA);
    } else {
        memcpy(w.data(), weights, sizeof(float) * P);
    }
    for (float x : w)
        if (!std::isfinite(x)) return bail(DOCK_E_INVALID_ARG);

    if (cudaMalloc(&ctx->d_rec, n_pad * sizeof(float)) != cudaSuccess) {
        cudaGetLastError();
        return bail(DOCK_E_OOM);
    }
    float* d_src = nullptr;
    bool rec_dev = rk == 1;
    if (rec_dev) {
        d_src = const_cast<float*>(receptor);
    } else {
        for (size_t i = 0; i < n_in; i++)
            if (!std::isfinite(receptor[i])) return bail(DOCK_E_INVALID_ARG);
        if (cudaMalloc(&d_src, n_in * sizeof(float)) != cudaSuccess) {
            cudaGetLastError();
            return bail(DOCK_E_OOM);
        }
        if (cudaMemcpyAsync(d_src, receptor, n_in * sizeof(float), cudaMemcpyHostToDevice, ctx->stream) !=
            cudaSuccess) {
            cudaFree(d_src);
            return bail(DOCK_E_CUDA);
        }
    }
    bool ok = cudaMalloc(&ctx->d_small, 64) == cudaSuccess && cudaHostAlloc(&ctx->h_small, 64, 0) == cudaSuccess &&
              cudaMalloc(&ctx->d_w, sizeof(float) * P) == cudaSuccess &&
              cudaMalloc(&ctx->d_eye, sizeof(float) * P * P) == cudaSuccess &&
              cudaMalloc(&ctx->d_ones, sizeof(float) * P) == cudaSuccess;
    if (!ok) {
        if (!rec_dev) cudaFree(d_src);
        cudaGetLastError();
        return bail(DOCK_E_OOM);
    }
    std::vector<float> eye((size_t)P * P, 0.f), ones(P, 1.f);
    for (int p = 0; p < P; p++) eye[(size_t)p * P + p] = 1.f;
    cudaMemcpy(ctx->d_w, w.data(), sizeof(float) * P, cudaMemcpyHostToDevice);
    cudaMemcpy(ctx->d_eye, eye.data(), sizeof(float) * P * P, cudaMemcpyHostToDevice);
    cudaMemcpy(ctx->d_ones, ones.data(), sizeof(float) * P, cudaMemcpyHostToDevice);
    cudaMemsetAsync(ctx->d_small, 0, 64, ctx->stream);
    // tcgen05 dynamic tile scheduler: [CTAs done, chunks taken per segment (< 2 n_sms segments)], zero
    // between launches (the last CTA of each launch resets it); without it variant 1 runs region mode
    if (cudaMalloc(&ctx->d_sched, sizeof(unsigned long long) * (2 * ctx->n_sms + 2)) == cudaSuccess)
        cudaMemsetAsync(ctx->d_sched, 0, sizeof(unsigned long long) * (2 * ctx->n_sms + 2), ctx->stream);
    else
        ctx->d_sched = nullptr;
    cudaGetLastError();
    if (rec_dev) {
        dk::k_count_nonfinite<<<1024, 256, 0, ctx->stream>>>(d_src, n_in, reinterpret_cast<unsigned*>(ctx->d_small));
    }
    dk::k_pad_receptor<<<2048, 256, 0, ctx->stream>>>(d_src, ctx->d_rec, ctx->nx, ctx->ny, ctx->nz, G.Xp, G.Yp,
                                                       G.Zp, P);
    // tcgen05 engine: bf16-split, channel-grouped, cyclic-halo copies of the receptor
    {
        ctx->tc_Gch = (P + 3) / 4;
        // variant 2 row width: the fewest wasted x translations (ties: 128, then 160, then 64)
        int best_w = 1 << 30;
        for (int ntt : {128, 160, 64}) {
            const int w = (ctx->nx + ntt - 1) / ntt * ntt;
            if (w < best_w) {
                best_w = w;
                ctx->tcs_ntt = ntt;
            }
        }
        const int q2 = tcs_q(ctx->tcs_ntt);
        const int ntx1 = (ctx->nx + tc::NT - 1) / tc::NT, ntx2 = (ctx->nx + ctx->tcs_ntt - 1) / ctx->tcs_ntt;
        int xp = 0;
        for (int mm = 1; mm <= ctx->m_max; mm++)
            xp = std::max({xp, (ntx1 - 1) * tc::NT + tc::pair_txb(mm, tc::NT),
                           (ntx2 - 1) * ctx->tcs_ntt + tc::pair_txb(mm, ctx->tcs_ntt)});
        ctx->tc_Xp = round_up(xp, 2);
        ctx->tc_Yp = std::max(round_up(ctx->ny, 4), round_up(ctx->ny, q2)) + ctx->m_max - 1;
        ctx->tc_Zp = ctx->nz + ctx->m_max - 1;
        const size_t bytes = (size_t)ctx->tc_Gch * ctx->tc_Zp * ctx->tc_Yp * ctx->tc_Xp * 16;
        if (cudaMalloc(&ctx->d_rec_tc, bytes) == cudaSuccess && cudaMalloc(&ctx->d_rec_pair, bytes) == cudaSuccess) {
            tc::k_pack_receptor_tc<<<2048, 256, 0, ctx->stream>>>(d_src, ctx->d_rec_tc, ctx->nx, ctx->ny, ctx->nz,
                                                                   ctx->tc_Xp, ctx->tc_Yp, ctx->tc_Zp, P, ctx->tc_Gch);
            tc::k_pack_receptor_pair_tc<<<2048, 256, 0, ctx->stream>>>(d_src, ctx->d_rec_pair, ctx->nx, ctx->ny,
                                                                        ctx->nz, ctx->tc_Xp, ctx->tc_Yp, ctx->tc_Zp, P,
                                                                        ctx->tc_Gch);
        } else {
            cudaGetLastError();
            cudaFree(ctx->d_rec_tc);
            ctx->d_rec_tc = nullptr;   // the tensor-core engine is then unavailable
            ctx->d_rec_pair = nullptr;
        }
    }
    cudaError_t e = cudaGetLastError();
    if (e == cudaSuccess) e = cudaMemcpyAsync(ctx->h_small, ctx->d_small, 16, cudaMemcpyDeviceToHost, ctx->stream);
    if (e == cudaSuccess) e = cudaStreamSynchronize(ctx->stream);
    if (!rec_dev) cudaFree(d_src);
    if (e != cudaSuccess) return bail(DOCK_E_CUDA);
    if (ctx->h_small[0] != 0) return bail(DOCK_E_INVALID_ARG);
    for (int m = 1; m <= ctx->m_max; m++) {
        dock_status s = make_plan(ctx, m);
        if (s != DOCK_OK && m == ctx->m_max) return bail(s);
        for (int v = 1; v <= 2; v++)
            if (make_tc_plan(ctx, m, v) != DOCK_OK) return bail(DOCK_E_CUDA);
    }
    *out = ctx;
    return DOCK_OK;
}

dock_status dock_set_tuning(dock_ctx* ctx, int key, int64_t value)
{
    if (!ctx) return DOCK_E_INVALID_ARG;
    switch (key) {
        case DOCK_TUNE_REGIONS:
            if (value < 0) return fail(ctx, DOCK_E_INVALID_ARG, "regions < 0");
            ctx->regions_override = (int)value;
            return DOCK_OK;
        case DOCK_TUNE_FORCE_FALLBACK: ctx->force_fallback = value ? 1 : 0; return DOCK_OK;
        case DOCK_TUNE_ENGINE:
            if (value < 0 || value > 4)
                return fail(ctx, DOCK_E_INVALID_ARG,
                            "engine must be 0 (auto), 1 (FFMA), 2 (tcgen05), 3 (FFT) or 4 (sparse ligand)");
            ctx->engine = (int)value;
            return DOCK_OK;
        case DOCK_TUNE_TC_VARIANT:
            if (value < 0 || value > 2) return fail(ctx, DOCK_E_INVALID_ARG, "tc variant must be 0, 1 or 2");
            ctx->tc_variant = (int)value;
            return DOCK_OK;
        case DOCK_TUNE_TC_EPILOGUE_WARPS:
            if (value != 0 && value != 4 && value != 8 && value != 16)
                return fail(ctx, DOCK_E_INVALID_ARG, "epilogue warps must be 0, 4, 8 or 16");
            ctx->tc_nepi = (int)value;
            return DOCK_OK;
        case DOCK_TUNE_TC_CHUNK:
            if (value < 0 || value > 4096) return fail(ctx, DOCK_E_INVALID_ARG, "tc chunk must be 0..4096");
            ctx->tc_chunk = (int)value;
            return DOCK_OK;
        case DOCK_TUNE_SHARD: {
            const int world = (int)(value >> 16), rank = (int)(value & 0xffff);
            if (world < 1 || world > 4096 || rank >= world)
                return fail(ctx, DOCK_E_INVALID_ARG, "shard: value = world << 16 | rank, 1 <= world, rank < world");
            ctx->shard_world = world;
            ctx->shard_rank = rank;
            return DOCK_OK;
        }
        case DOCK_TUNE_TC_SCHEDULE:
            if (value < 0 || value > 2) return fail(ctx, DOCK_E_INVALID_ARG, "tc schedule must be 0, 1 or 2");
            ctx->tc_sched = (int)value;
            return DOCK_OK;
        case DOCK_TUNE_CAND_CAP:
            if (value < 32 || value > (1 << 20)) return fail(ctx, DOCK_E_INVALID_ARG, "cand cap out of range");
            ctx->cand_cap = (int)value;
            return DOCK_OK;
    }
    return fail(ctx, DOCK_E_INVALID_ARG, "unknown tuning key %d", key);
}

dock_status dock_get_info(const dock_ctx* ctx, dock_info* info)
{
    if (!ctx || !info) return DOCK_E_INVALID_ARG;
    memset(info, 0, sizeof(*info));
    info->lanes_x = ctx->geo.LX;
    info->tile_x = ctx->geo.TX;
    info->tile_y = ctx->geo.TY;
    info->tile_z = ctx->geo.TZ;
    info->n_tiles = ctx->geo.ntiles;
    const MPlan& pl = ctx->plan[ctx->m_max];
    info->n_stages = pl.nstage;
    info->smem_bytes = pl.smem;
    info->regions_last = ctx->regions_last;
    info->items_last = ctx->items_last;
    info->fallback_last = ctx->fallback_last;
    info->cand_max_last = ctx->cand_max_last;
    info->kernels_last = ctx->kernels_last;
    info->rot_batch = dk::RB;
    info->x_per_thread = dk::XT;
    info->padded_x = ctx->geo.Xp;
    info->padded_y = ctx->geo.Yp;
    info->padded_z = ctx->geo.Zp;
    info->l2_bytes = ctx->l2_bytes;
    info->corr_ms_last = -1.0;
    if (ctx->ev_corr_valid) {
        float ms = 0.f;
        if (cudaEventElapsedTime(&ms, ctx->ev_corr[0], ctx->ev_corr[1]) == cudaSuccess) info->corr_ms_last = ms;
        else cudaGetLastError();
    }
    info->n_sms = ctx->n_sms;
    info->engine_last = ctx->engine_last;
    info->tc_available = (ctx->tcplan[1][ctx->m_max].ok || ctx->tcplan[2][ctx->m_max].ok) ? 1 : 0;
    info->tc_variant_last = ctx->tc_variant_last;
    info->tc_ksteps_last = ctx->tc_ksteps_last;
    if (ctx->tc_variant_last > 0) {
        const TcPlan& tp = ctx->tcplan[ctx->tc_variant_last][ctx->tc_m_last];
        info->tc_row_last = tp.ntt;
        info->tc_rows_per_tile_last = tp.q;
    }
    info->pending = ctx->unsynced ? 1 : 0;
    if (ctx->unsynced && ctx->ev_done && cudaEventQuery(ctx->ev_done) == cudaSuccess) {
        // the last call has completed: its statistics are readable without a sync point
        info->pending = 0;
        info->fallback_last = (unsigned)ctx->h_small[1];
        info->cand_max_last = (unsigned)ctx->h_small[2];
    }
    cudaGetLastError();
    info->fb_chunk = fb_chunk(ctx, ctx->engine_last);
    info->sp_atom_grids_last = ctx->sp_natoms_last;
    info->sp_terms_last = ctx->sp_terms_last;
    if (ctx->engine_last == ENG_SPARSE) {
        info->sp_row_last = ctx->sp_tx_last;
        info->sp_zt_last = ctx->sp_zt_last;
    }
    info->tc_ksteps_exec_last = -1.0;
    if (ctx->tc_variant_last == 1 && ctx->tc_blocks_last > 0 && !info->pending)
        info->tc_ksteps_exec_last = double((unsigned)ctx->h_small[3]) / ctx->tc_blocks_last;
    return DOCK_OK;
}

dock_status dock_probe_batch(dock_ctx* ctx, const dock_probe_desc* probes, int n_probes, const double* rot,
                             int n_rot, int64_t unit_begin, int64_t unit_end, int k, int rho, dock_pose* out)
{
    TRY(check_ctx(ctx));
    ctx->kernels_last = 0;
    ctx->ev_corr_valid = false;
    if (!rot || !out || n_rot < 1) return fail(ctx, DOCK_E_INVALID_ARG, "null rotations/output or n_rot < 1");
    if (k < 1) return fail(ctx, DOCK_E_INVALID_ARG, "k < 1");
    if (k > DOCK_MAX_K) return fail(ctx, DOCK_E_UNSUPPORTED, "k > %d", DOCK_MAX_K);
    if (rho < 0 || 2 * rho + 1 > std::min(ctx->nx, std::min(ctx->ny, ctx->nz)))
        return fail(ctx, DOCK_E_INVALID_ARG, "rho out of range");
    const double ball = std::pow(2.0 * rho + 1.0, 3);
    if ((double)k * ball > (double)ctx->nx * ctx->ny * ctx->nz)
        return fail(ctx, DOCK_E_INVALID_ARG, "k*(2rho+1)^3 exceeds the number of translations");
    int m = 0;
    TRY(validate_probes(ctx, probes, n_probes, &m));
    if (unit_begin < 0 || unit_end < unit_begin || unit_end > (int64_t)n_probes * n_rot)
        return fail(ctx, DOCK_E_INVALID_ARG, "bad unit range");
    const int64_t n_units64 = unit_end - unit_begin;
    // 32-bit index math of the per-call kernels: (units rounded to RB) * P must fit in an int
    if (n_units64 > (int64_t)1 << 28 || (n_units64 + dk::RB) * ctx->P > 0x7fffffffLL)
        return fail(ctx, DOCK_E_UNSUPPORTED, "too many units in one call");
    const int n_units = (int)n_units64;
    bool out_dev = false, rot_dev = false;
    PTR_KIND(out_dev, out, "out");
    PTR_KIND(rot_dev, rot, "rot");
    if (n_units == 0) return out_dev ? DOCK_OK : sync_point(ctx);
    TRY(make_plan(ctx, m));
    if (!rot_dev) {
        for (int64_t i = 0; i < (int64_t)9 * n_rot; i++)
            if (!std::isfinite(rot[i])) return fail(ctx, DOCK_E_INVALID_ARG, "non-finite rotation");
    }
    const int P = ctx->P, m3 = m * m * m;
    const int64_t n_batches = (n_units + dk::RB - 1) / dk::RB;
    const int cap = ctx->cand_cap;
    TRY(ensure(ctx, ctx->Lw, sizeof(float) * n_batches * P * m3 * dk::RB));
    TRY(ensure(ctx, ctx->T, sizeof(unsigned long long) * n_units));
    TRY(ensure(ctx, ctx->mu, sizeof(unsigned long long) * n_units));
    TRY(ensure(ctx, ctx->cnt, sizeof(unsigned int) * n_units));
    TRY(ensure(ctx, ctx->cand, sizeof(unsigned long long) * (size_t)n_units * cap));
    TRY(ensure(ctx, ctx->fb_list, sizeof(int) * n_units));
    void* d_poses = out;
    if (!out_dev) {
        TRY(ensure(ctx, ctx->poses, sizeof(dock_pose) * (size_t)n_units * k));
        d_poses = ctx->poses.p;
    }
    // engine; the direct engines' fallback buffers exist before staging (their addresses travel in dk::FbDyn)
    int kind = ENG_FFT;
    SpCall sc;
    if (ctx->engine != 3) {
        if (ctx->engine == 0 || ctx->engine == 4)
            TRY(sp_prepare(ctx, m, probes, n_probes, n_rot, unit_begin, unit_end, &sc));
        TRY(select_engine(ctx, m, sc.ok, sp_better(ctx, sc, m, n_units), &kind));
        if (ctx->shard_world > 1 && kind != ENG_TC)
            return fail(ctx, DOCK_E_UNSUPPORTED, "block sharding needs the tcgen05 variant-1 engine");
        TRY(fb_buffers(ctx, m, fb_chunk(ctx, kind), k));
    }
    const bool use_tc = kind == ENG_TC;
    dk::FbDyn fb = fb_template(ctx, m, fb_chunk(ctx, kind), unit_begin, n_rot, d_poses);
    const double *d_xyz, *d_rot;
    const float* d_coef;
    const int* d_off;
    const dk::FbDyn* d_fb = nullptr;
    const void* d_groups = nullptr;
    TRY(stage_inputs(ctx, probes, n_probes, rot, n_rot, &d_xyz, &d_coef, &d_off, &d_rot, &fb, &d_fb,
                     kind == ENG_SPARSE ? sc.groups.data() : nullptr,
                     kind == ENG_SPARSE ? sizeof(sp::Group) * sc.groups.size() : 0, &d_groups));

    unsigned int* fb_cnt = reinterpret_cast<unsigned int*>(ctx->d_small + 1);
    unsigned int* cand_max = reinterpret_cast<unsigned int*>(ctx->d_small + 2);
    dk::k_reset<<<(n_units + 255) / 256, 256, 0, ctx->stream>>>(
        static_cast<unsigned long long*>(ctx->T.p), static_cast<unsigned long long*>(ctx->mu.p),
        static_cast<unsigned int*>(ctx->cnt.p), n_units, fb_cnt, cand_max, reinterpret_cast<unsigned*>(ctx->d_small + 3));
    CU(cudaGetLastError());
    ctx->kernels_last++;

    // a1: voxelize (+ rotation / box validation; errors are sticky device status bits)
    if (kind == ENG_SPARSE)
        TRY(sp_run_pre(ctx, sc, n_units, unit_begin, n_rot, d_xyz, d_coef, d_off, d_rot, ctx->d_w));
    else
        TRY(run_voxelize(ctx, m, n_units, unit_begin, nullptr, n_rot, d_xyz, d_coef, d_off, d_rot, ctx->d_w,
                         static_cast<float*>(ctx->Lw.p)));

    if (ctx->engine == 3) {
        // comparison engine: FFT score grids + exact greedy (no fused top-k, no fallback needed); this engine
        // synchronises internally (host-driven chunking), whatever the output memory
        ctx->engine_last = 3;
        ctx->tc_variant_last = 0;
        CU(cudaEventRecord(ctx->ev_corr[0], ctx->stream));
        TRY(run_fft_poses(ctx, m, n_units, unit_begin, n_rot, k, rho, d_poses));
        CU(cudaEventRecord(ctx->ev_corr[1], ctx->stream));
        ctx->ev_corr_valid = true;
        if (!out_dev)
            CU(cudaMemcpyAsync(out, d_poses, sizeof(dock_pose) * (size_t)n_units * k, cudaMemcpyDeviceToHost,
                               ctx->stream));
        TRY(end_call(ctx));
        return sync_point(ctx);
    }

    // a2-a5: correlation + fused weighted score + on-chip top-k lists (no score grid in HBM)
    auto* Tp = static_cast<unsigned long long*>(ctx->T.p);
    auto* mup = static_cast<unsigned long long*>(ctx->mu.p);
    auto* cntp = static_cast<unsigned int*>(ctx->cnt.p);
    auto* candp = static_cast<unsigned long long*>(ctx->cand.p);
    if (kind == ENG_SPARSE) {
        const int64_t n_groups = (int64_t)sc.groups.size();
        sp::SpArgs a = sp_args(ctx, sc, static_cast<const sp::Group*>(d_groups), n_groups);
        a.k = k;
        a.rho = rho;
        a.cap = cap;
        a.T = Tp;
        a.mu = mup;
        a.cnt = cntp;
        a.cand = candp;
        const int64_t items = n_groups * a.G;
        if (items > 0x7fffffff) return fail(ctx, DOCK_E_UNSUPPORTED, "too many work items");
        CU(cudaEventRecord(ctx->ev_corr[0], ctx->stream));
        CU(dock_launch_sparse(sc.xts, sc.zt, false, ctx->sp_tmap, sc.smem, a, (int)items, ctx->stream));
        CU(cudaEventRecord(ctx->ev_corr[1], ctx->stream));
        ctx->regions_last = a.G;
        ctx->items_last = items;
    } else if (use_tc) {
        const int64_t n_blocks = (n_units + tc::ROT - 1) / tc::ROT;
        int v = 0, G = 0;
        if (!plan_tc_launch(ctx, m, n_units, &v, &G)) return fail(ctx, DOCK_E_UNSUPPORTED, "no tensor-core plan");
        TRY(pack_weights_tc(ctx, m, v, n_units, static_cast<const float*>(ctx->Lw.p), false, nullptr, true));
        ctx->tc_variant_last = v;
        if (ctx->shard_world > 1 && v != 1)
            return fail(ctx, DOCK_E_UNSUPPORTED, "block sharding needs the tcgen05 variant-1 engine");
        ctx->tc_ksteps_last = ctx->tcplan[v][m].nsteps;
        ctx->tc_m_last = m;
        tc::TcArgs ta = tc_args(ctx, m, v, n_units, G, static_cast<const unsigned char*>(ctx->Wtc.p));
        ta.k = k;
        ta.rho = rho;
        ta.cap = cap;
        ta.T = Tp;
        ta.mu = mup;
        ta.cnt = cntp;
        ta.cand = candp;
        const int64_t items = tc_ctas(ta, n_units, ctx->n_sms);
        if (items > 0x7fffffff) return fail(ctx, DOCK_E_UNSUPPORTED, "too many work items");
        if (v == 1 && ta.chunk > 0 && ctx->tc_sched != 2 && n_blocks <= (1 << 16) && items > 0) {
            // scheduler segments of equal estimated cost (blocks' occupancy schedules differ in length)
            TRY(ensure(ctx, ctx->tc_seg, sizeof(long long) * (items + 1)));
            TRY(ensure(ctx, ctx->tc_pref, sizeof(long long) * n_blocks));
            const int cpb = (ta.ntiles + ta.chunk - 1) / ta.chunk;
            tc::k_tc_segments<<<1, 256, 0, ctx->stream>>>(ta.kinfo, ta.blkmap, ta.blkmap ? ta.n_blocks : (int)n_blocks,
                                                          cpb, (int)items, ctx->tc_seg_cost,
                                                          static_cast<long long*>(ctx->tc_pref.p),
                                                          static_cast<long long*>(ctx->tc_seg.p));
            CU(cudaGetLastError());
            ctx->kernels_last++;
            ta.seg = static_cast<const long long*>(ctx->tc_seg.p);
        }
        if (ctx->d_trace) CU(cudaMemsetAsync(ctx->d_trace, 0, sizeof(unsigned long long) * tc::TR_N, ctx->stream));
        CU(cudaEventRecord(ctx->ev_corr[0], ctx->stream));
        if (items > 0) CU(launch_tc(m, v, false, ctx->tcplan[v][m], ta, (int)items, ctx->stream));   // 0: no block here
        CU(cudaEventRecord(ctx->ev_corr[1], ctx->stream));
        if (ctx->d_trace) {
            std::vector<unsigned long long> hv(tc::TR_N);
            unsigned long long* h = hv.data();
            CU(cudaMemcpyAsync(h, ctx->d_trace, sizeof(unsigned long long) * tc::TR_N, cudaMemcpyDeviceToHost,
                               ctx->stream));
            CU(cudaStreamSynchronize(ctx->stream));
            if (const char* f = getenv("DOCK_TC_TRACE_CTAS")) {   // per-CTA start / end / SM id dump
                if (FILE* fp = fopen(f, "w")) {
                    for (int i = 0; i < (int)std::min<int64_t>(items, tc::TR_MAXCTA); i++)
                        fprintf(fp, "%d %llu %llu %llu\n", i, h[tc::TR_CTA0 + 3 * i], h[tc::TR_CTA0 + 3 * i + 1],
                                h[tc::TR_CTA0 + 3 * i + 2]);
                    fclose(fp);
                }
            }
            const double c = h[tc::TR_CTAS] ? double(h[tc::TR_CTAS]) : 1.0;
            const double e = h[tc::TR_EPI_WARPS] ? double(h[tc::TR_EPI_WARPS]) : 1.0;
            fprintf(stderr,
                    "TCTRACE {\"variant\": %d, \"ctas\": %llu, \"tiles_per_cta\": %.1f, "
                    "\"mma_total\": %.0f, \"mma_wait_tmem_empty\": %.0f, \"mma_wait_w_full\": %.0f, "
                    "\"mma_wait_rec_full\": %.0f, \"epi_total\": %.0f, \"epi_wait_tm_full\": %.0f, "
                    "\"epi_ldtm\": %.0f, \"prod_total\": %.0f, \"prod_wait_w_empty\": %.0f, "
                    "\"prod_wait_rec_empty\": %.0f, \"span_ms\": %.4f, \"cta_ms\": %.4f, "
                    "\"epi_wait_chunk\": %.0f, \"mma_wait_chunk\": %.0f, \"rec_wait_chunk\": %.0f, "
                    "\"epi_publish\": %.0f, \"inserts_per_tile_lane\": %.3f, \"gates_per_tile_lane\": %.3f, "
                    "\"rare_entries_per_tile_warp\": %.3f}\n",
                    v, h[tc::TR_CTAS], h[tc::TR_TILES] / c, h[tc::TR_MMA_TOTAL] / c,
                    h[tc::TR_MMA_TMEMPTY] / c, h[tc::TR_MMA_WFULL] / c, h[tc::TR_MMA_RFULL] / c,
                    h[tc::TR_EPI_TOTAL] / e, h[tc::TR_EPI_TMFULL] / e, h[tc::TR_EPI_LDTM] / e,
                    h[tc::TR_PROD_TOTAL] / c, h[tc::TR_PROD_WEMPTY] / c, h[tc::TR_PROD_REMPTY] / c,
                    h[tc::TR_GT_END] ? (h[tc::TR_GT_END] - ~h[tc::TR_GT_START_NOT]) * 1e-6 : 0.0,
                    h[tc::TR_GT_CTA_NS] * 1e-6 / c, h[tc::TR_EPI_CHWAIT] / e, h[tc::TR_MMA_CHWAIT] / c,
                    h[tc::TR_REC_CHWAIT] / c, h[tc::TR_EPI_PUB] / e,
                    h[tc::TR_TILES] ? h[tc::TR_EPI_INS] / (double(h[tc::TR_TILES]) * tc::ROT) : 0.0,
                    h[tc::TR_TILES] ? h[tc::TR_EPI_GATE] / (double(h[tc::TR_TILES]) * tc::ROT) : 0.0,
                    h[tc::TR_TILES] ? h[tc::TR_EPI_WRARE] / (double(h[tc::TR_TILES]) * ta.nepi) : 0.0);
        }
        ctx->regions_last = ta.chunk > 0 ? 0 : G;
        ctx->items_last = items;
    } else {
        const int G = choose_regions(ctx, n_batches);
        dk::CorrArgs a = corr_args(ctx, m, n_units, G, static_cast<const float*>(ctx->Lw.p));
        a.k = k;
        a.rho = rho;
        a.T = Tp;
        a.mu = mup;
        a.cnt = cntp;
        a.cand = candp;
        a.cap = cap;
        const int64_t items = n_batches * G;
        if (items > 0x7fffffff) return fail(ctx, DOCK_E_UNSUPPORTED, "too many work items");
        CU(cudaEventRecord(ctx->ev_corr[0], ctx->stream));
        CU(dock_launch_ffma(m, false, ctx->plan[m].tmap, ctx->plan[m].smem, a, (int)items, ctx->stream));
        CU(cudaEventRecord(ctx->ev_corr[1], ctx->stream));
        ctx->regions_last = G;
        ctx->items_last = items;
    }
    ctx->ev_corr_valid = true;
    ctx->kernels_last++;

    // a6: per-rotation merge + greedy filter
    dk::MergeArgs ma{};
    ma.n_slots = n_units;
    ma.k = k;
    ma.rho = rho;
    ma.cap = cap;
    ma.n_rot = n_rot;
    ma.nx = ctx->nx;
    ma.ny = ctx->ny;
    ma.nz = ctx->nz;
    ma.unit_begin = unit_begin;
    ma.cand = candp;
    ma.cnt = cntp;
    ma.mu = mup;
    ma.force_fallback = ctx->force_fallback;
    ma.poses = d_poses;
    ma.fb_list = static_cast<int*>(ctx->fb_list.p);
    ma.fb_cnt = fb_cnt;
    ma.cand_max = cand_max;
    ma.owned = (use_tc && ctx->tc_nblk_local >= 0) ? static_cast<const unsigned char*>(ctx->tc_owned.p) : nullptr;
    dk::k_merge<<<(n_units + 7) / 8, 256, 0, ctx->stream>>>(ma);
    CU(cudaGetLastError());
    ctx->kernels_last++;

    // a6': exact fallback of the flagged rotations, driven by the device-side flag count
    TRY(launch_fallback(ctx, m, kind, k, rho, d_fb, &sc));

    // a7: output.  Device output: return now (results and errors at dock_sync / the next sync point);
    // host output: copy back and synchronise.
    if (!out_dev)
        CU(cudaMemcpyAsync(out, d_poses, sizeof(dock_pose) * (size_t)n_units * k, cudaMemcpyDeviceToHost,
                           ctx->stream));
    TRY(end_call(ctx));
    return out_dev ? DOCK_OK : sync_point(ctx);
}

dock_status dock_sync(dock_ctx* ctx)
{
    TRY(check_ctx(ctx));
    return sync_point(ctx);
}

dock_status dock_probe(dock_ctx* ctx, const dock_probe_desc* probe, const double* rot, int n_rot, int k, int rho,
                       dock_pose* out)
{
    return dock_probe_batch(ctx, probe, 1, rot, n_rot, 0, n_rot, k, rho, out);
}

dock_status dock_score_grid(dock_ctx* ctx, const dock_probe_desc* probe, const double* rot9, float* out,
                            float* per_term)
{
    TRY(check_ctx(ctx));
    ctx->kernels_last = 0;
    if (!rot9 || !out) return fail(ctx, DOCK_E_INVALID_ARG, "null rotation/output");
    int m = 0;
    TRY(validate_probes(ctx, probe, 1, &m));
    TRY(make_plan(ctx, m));
    int kind = ENG_FFT;
    SpCall sc;
    if (ctx->engine != 3) {
        if (ctx->engine == 0 || ctx->engine == 4) TRY(sp_prepare(ctx, m, probe, 1, 1, 0, 1, &sc));
        TRY(select_engine(ctx, m, sc.ok, sp_better(ctx, sc, m, 1), &kind));
    } else {
        ctx->engine_last = 3;
    }
    const double *d_xyz, *d_rot;
    const float* d_coef;
    const int* d_off;
    const void* d_groups = nullptr;
    TRY(stage_inputs(ctx, probe, 1, rot9, 1, &d_xyz, &d_coef, &d_off, &d_rot, nullptr, nullptr,
                     kind == ENG_SPARSE ? sc.groups.data() : nullptr,
                     kind == ENG_SPARSE ? sizeof(sp::Group) * sc.groups.size() : 0, &d_groups));
    const size_t ncell = (size_t)ctx->nx * ctx->ny * ctx->nz;
    const int m3 = m * m * m;
    TRY(ensure(ctx, ctx->Lw, sizeof(float) * ctx->P * m3 * dk::RB));
    bool out_dev = false, pt_dev = false;
    PTR_KIND(out_dev, out, "out");
    PTR_KIND(pt_dev, per_term, "per_term");
    size_t need = (out_dev ? 0 : ncell) + (per_term && !pt_dev ? ncell * ctx->P : 0);
    if (need) TRY(ensure(ctx, ctx->grid, sizeof(float) * need));
    float* g_out = out_dev ? out : static_cast<float*>(ctx->grid.p);
    float* g_pt = per_term ? (pt_dev ? per_term : static_cast<float*>(ctx->grid.p) + (out_dev ? 0 : ncell)) : nullptr;
    // one score grid with weights w (folded into L, or into the atom grids of the sparse engine)
    auto grid_fn = [&](const float* w, float* dst) -> dock_status {
        if (kind == ENG_SPARSE) {
            TRY(sp_run_pre(ctx, sc, 1, 0, 1, d_xyz, d_coef, d_off, d_rot, w));
            sp::SpArgs a = sp_args(ctx, sc, static_cast<const sp::Group*>(d_groups), 1);
            a.grid = dst;
            CU(dock_launch_sparse(sc.xts, sc.zt, true, ctx->sp_tmap, sc.smem, a, a.G, ctx->stream));
            ctx->kernels_last++;
            return DOCK_OK;
        }
        TRY(run_voxelize(ctx, m, 1, 0, nullptr, 1, d_xyz, d_coef, d_off, d_rot, w, static_cast<float*>(ctx->Lw.p)));
        if (kind == ENG_FFT) return run_grid_fft(ctx, m, 0, 1, static_cast<const float*>(ctx->Lw.p), dst);
        return kind == ENG_TC ? run_grid_tc(ctx, m, 1, static_cast<const float*>(ctx->Lw.p), dst)
                              : run_grid(ctx, m, 1, static_cast<const float*>(ctx->Lw.p), dst);
    };
    TRY(grid_fn(ctx->d_w, g_out));
    if (per_term)
        for (int p = 0; p < ctx->P; p++) TRY(grid_fn(ctx->d_eye + (size_t)p * ctx->P, g_pt + ncell * p));
    if (!out_dev) CU(cudaMemcpyAsync(out, g_out, sizeof(float) * ncell, cudaMemcpyDeviceToHost, ctx->stream));
    if (per_term && !pt_dev)
        CU(cudaMemcpyAsync(per_term, g_pt, sizeof(float) * ncell * ctx->P, cudaMemcpyDeviceToHost, ctx->stream));
    TRY(end_call(ctx));
    return sync_point(ctx);
}

dock_status dock_voxelize(dock_ctx* ctx, const dock_probe_desc* probe, const double* rot, int n_rot, float* out)
{
    TRY(check_ctx(ctx));
    ctx->kernels_last = 0;
    ctx->ev_corr_valid = false;
    if (!rot || !out || n_rot < 1) return fail(ctx, DOCK_E_INVALID_ARG, "null rotation/output");
    int m = 0;
    TRY(validate_probes(ctx, probe, 1, &m));
    const double *d_xyz, *d_rot;
    const float* d_coef;
    const int* d_off;
    TRY(stage_inputs(ctx, probe, 1, rot, n_rot, &d_xyz, &d_coef, &d_off, &d_rot));
    const int m3 = m * m * m, P = ctx->P;
    const int64_t nb = (n_rot + dk::RB - 1) / dk::RB;
    TRY(ensure(ctx, ctx->Lw, sizeof(float) * nb * P * m3 * dk::RB));
    bool out_dev = false;
    PTR_KIND(out_dev, out, "out");
    const size_t n_out = (size_t)n_rot * P * m3;
    if ((int64_t)n_rot * P * m3 + (int64_t)dk::RB * P * m3 > 0x7fffffffLL)
        return fail(ctx, DOCK_E_UNSUPPORTED, "too many rotations in one call");
    if (!out_dev) TRY(ensure(ctx, ctx->grid, sizeof(float) * n_out));
    float* g_out = out_dev ? out : static_cast<float*>(ctx->grid.p);
    TRY(run_voxelize(ctx, m, n_rot, 0, nullptr, n_rot, d_xyz, d_coef, d_off, d_rot, ctx->d_ones,
                     static_cast<float*>(ctx->Lw.p)));
    int n = (int)n_out;
    dk::k_unpack_L<<<(n + 255) / 256, 256, 0, ctx->stream>>>(static_cast<const float*>(ctx->Lw.p), g_out, n_rot, P,
                                                              m3);
    CU(cudaGetLastError());
    if (!out_dev) CU(cudaMemcpyAsync(out, g_out, sizeof(float) * n_out, cudaMemcpyDeviceToHost, ctx->stream));
    TRY(end_call(ctx));
    return sync_point(ctx);
}

}  // extern "C"

/*
 * dock.h -- C ABI of the B200-native rigid-docking hot path (libdock.so).
 *
 * Method: Sukhwani & Herbordt, "Fast Binding Site Mapping using GPUs and CUDA",
 * IPPS/IPDPS 2010 (dblp conf/ipps/SukhwaniH10).  "P:L<a>-<b>" cites PAPER.md lines.
 *
 * For every rotation of a small probe molecule, the probe is voxelized onto one
 * m^3 grid per energy term, each grid is direct-correlated against
 * the matching precomputed receptor grid (Eq. 1; direct correlation
 * P:L503-509), the terms are summed with their weights (Eq. 2) and
 * the best translations are kept per rotation by "selecting the best score and
 * then excluding its neighbors while selecting the next best score"
 * (Fig. 5); FTMap keeps 4 per rotation.
 *
 * Readings of the paper where it is silent:
 *   - score   S_r[t] = sum_p w_p sum_{v in [0,m)^3} L_{r,p}[v] R_p[(t+v) mod n]
 *             (cyclic boundary, Q1/Q2); best = MINIMUM weighted energy (Q7);
 *   - voxelize g = (Q x)/h + (m-1)/2, v = floor(g + 0.5) in FP64, coefficients of
 *             atoms sharing a voxel are summed, an atom outside [0,m)^3 is an error (Q3);
 *   - filter  keys (score, t_lin) ascending, -0.0 == +0.0 (Q8); exclusion = cyclic
 *             Chebyshev ball of radius rho around each pick (Q9: rho = 1 is the
 *             paper-faithful default, rho = 0 is plain top-k).
 *   - t_lin = (tz*ny + ty)*nx + tx; x is the fastest axis everywhere.
 * GPU arithmetic (reading Q15): engine 1 is FP32 FFMA; the default tcgen05 engine multiplies bf16
 * hi/lo splits of both operands (x = hi + lo, bf16x3: Rhi*Whi + Rlo*Whi + Rhi*Wlo) and accumulates
 * in FP32 -- the dropped Rlo*Wlo and the lo roundings bound the error by ~3*2^-18 relative per term,
 * i.e. ~1e-5*A against the 1e-4*A tolerance (reading Q16); integer-valued inputs stay exact.  The
 * FP64 oracle (oracle/) is the reference.
 *
 * Conventions
 *   - Every call returns dock_status (DOCK_OK = 0); no exception crosses the ABI.
 *   - Pointers may be host or device memory unless stated; the kind is detected with
 *     cudaPointerGetAttributes.  The library never takes ownership of caller memory:
 *     dock_init copies the receptor and weights; probe/rotation inputs are only read
 *     during the call.
 *   - All work runs on the context's stream.  dock_probe / dock_probe_batch with a DEVICE
 *     output pointer are asynchronous: they enqueue the whole hot path (including the exact
 *     fallback, whose loop is driven by a device-side flag count) and return without any host
 *     synchronisation; the poses are valid once the context's stream reaches that point (e.g.
 *     after dock_sync, or for any later work ordered on the stream such as an NCCL all-gather).
 *     Device-detected input errors (DOCK_E_BAD_ROTATION, DOCK_E_PROBE_OUTSIDE_GRID) of an
 *     asynchronous call are sticky and reported by the next sync point: dock_sync, or the next
 *     call with host output / dock_score_grid / dock_voxelize.  Calls with HOST output (and the
 *     debug calls) synchronise the stream before returning.
 *   - A context is bound to one device and one stream and is not thread-safe.
 *     After DOCK_E_CUDA the context is unusable and must be destroyed.
 */
#ifndef B200_DOCK_H
#define B200_DOCK_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef enum {
    DOCK_OK = 0,
    DOCK_E_INVALID_ARG = -1,        /* null pointer, dims < 1, k < 1, rho < 0, 2*rho+1 > min(n),
                                       k*(2rho+1)^3 > nx*ny*nz, bad unit range, non-finite input */
    DOCK_E_UNSUPPORTED = -2,        /* m > m_max or m > DOCK_MAX_M, n_terms > DOCK_MAX_TERMS,
                                       k > DOCK_MAX_K, probes of different m in one batch, grid too large */
    DOCK_E_PROBE_OUTSIDE_GRID = -3, /* an atom voxelizes outside [0,m)^3 for some rotation */
    DOCK_E_BAD_ROTATION = -4,       /* |Q^T Q - I| > 1e-9 (elementwise) or det(Q) <= 0 */
    DOCK_E_CUDA = -5,               /* CUDA runtime/driver failure; context unusable */
    DOCK_E_OOM = -6                 /* device allocation failed */
} dock_status;

#define DOCK_MAX_TERMS 32  /* P <= 32 correlation terms (the paper: up to 22) */
#define DOCK_MAX_M 8       /* probe grid edge m <= 8 (paper: <= 8^3 in constant memory) */
#define DOCK_MAX_K 32      /* poses kept per rotation (FTMap: 4) */

/* Engines (DOCK_TUNE_ENGINE) */
#define DOCK_ENGINE_AUTO 0
#define DOCK_ENGINE_FFMA 1
#define DOCK_ENGINE_TC 2
#define DOCK_ENGINE_FFT 3
#define DOCK_ENGINE_SPARSE 4

/* Pose flags */
#define DOCK_POSE_FALLBACK 1u   /* exact full-grid fallback was used for this rotation */
#define DOCK_POSE_EMPTY 2u      /* fewer than k translations were available (never with valid args) */

typedef struct dock_ctx dock_ctx;  /* opaque; owns all device memory of one receptor */

/* One kept pose: rotation index (into the rotation set), translation, weighted score. 16 B. */
typedef struct {
    int32_t rot;     /* rotation index r in [0, n_rot) */
    int32_t t_lin;   /* translation (tz*ny + ty)*nx + tx, -1 if none */
    float score;     /* S_r[t] in FP32 (the GPU value; oracle comparison within 1e-4*A) */
    uint32_t flags;  /* DOCK_POSE_* */
} dock_pose;

/* Receptor grid description (dock_init). */
typedef struct {
    int nx, ny, nz;   /* receptor grid / translation space, each >= 1 */
    int n_terms;      /* P, number of correlation terms (channels), 1..DOCK_MAX_TERMS */
    int m_max;        /* largest probe grid edge that will be docked, 1..DOCK_MAX_M */
    int device;       /* CUDA device ordinal */
    double spacing;   /* grid spacing h in Angstrom (> 0, finite); BASELINE uses 0.8.  double so that the
                         kernel divides by exactly the caller's h, as the FP64 oracle does (reading Q18) */
    void* stream;     /* cudaStream_t to run on (cudaStreamLegacy / cudaStreamPerThread allowed); NULL => the
                         context creates its own non-blocking stream (work of other streams is then NOT ordered
                         with the context's: the caller synchronises) */
} dock_grid_desc;

/* One probe (small molecule). */
typedef struct {
    int n_atoms;          /* >= 0 */
    int m;                /* probe grid edge, 1..m_max */
    const double* xyz;    /* [n_atoms][3] Angstrom, relative to the rotation centre; host or device */
    const float* coef;    /* [n_atoms][n_terms] per-atom per-term coefficient; host or device */
} dock_probe_desc;

/* dock_init -- copy the receptor grids and term weights to the device (once).
 *   receptor : [P][nz][ny][nx] float32 (x fastest), host or device; must be finite.
 *   weights  : [P] float32 term weights w_p of Eq. 2, host or device; finite.
 *   out      : receives the new context.
 * Builds the cyclic-halo padded copy and the TMA descriptors.  Not part of the hot path. */
dock_status dock_init(const dock_grid_desc* g, const float* receptor, const float* weights, dock_ctx** out);

/* dock_probe -- dock one probe over a rotation set.
 *   rot  : [n_rot][9] float64 row-major rotation matrices, host or device.
 *   k    : poses kept per rotation, 1..DOCK_MAX_K;  rho : exclusion radius >= 0.
 *   out  : [n_rot][k] dock_pose, host or device, caller-allocated.  Poses of one rotation
 *          are in pick order (ascending key).
 * Equivalent to dock_probe_batch(ctx, probe, 1, rot, n_rot, 0, n_rot, k, rho, out). */
dock_status dock_probe(dock_ctx* ctx, const dock_probe_desc* probe, const double* rot, int n_rot,
                       int k, int rho, dock_pose* out);

/* dock_probe_batch -- the hot path: dock the (probe, rotation) units
 * [unit_begin, unit_end) of the probe-major unit space (unit = probe*n_rot + r).
 * This is the shard entry point for multi-GPU runs (each rank passes its range).
 *   probes : [n_probes] host array of descriptors; all probes must have the same m.
 *   out    : [(unit_end-unit_begin)][k] dock_pose, host or device. */
dock_status dock_probe_batch(dock_ctx* ctx, const dock_probe_desc* probes, int n_probes,
                             const double* rot, int n_rot, int64_t unit_begin, int64_t unit_end,
                             int k, int rho, dock_pose* out);

/* dock_sync -- sync point of the asynchronous calls: waits for the context's stream, returns the
 * first device-detected error of the calls since the previous sync point (DOCK_E_BAD_ROTATION,
 * DOCK_E_PROBE_OUTSIDE_GRID; cleared by this call) or DOCK_E_CUDA, and makes the last call's
 * statistics (fallback_last, cand_max_last) available to dock_get_info. */
dock_status dock_sync(dock_ctx* ctx);

/* dock_score_grid -- test/debug: the full weighted score grid of one rotated probe.
 *   rot9     : [9] float64 rotation, host or device.
 *   out      : [nz][ny][nx] float32 S (weighted), host or device.
 *   per_term : optional [P][nz][ny][nx] float32 unweighted C_p (w = e_p); may be NULL.
 * Uses the same correlation kernel as the hot path (grid epilogue instead of top-k). */
dock_status dock_score_grid(dock_ctx* ctx, const dock_probe_desc* probe, const double* rot9,
                            float* out, float* per_term);

/* dock_voxelize -- test/debug: the rotated, voxelized probe grids (unweighted L, FP32).
 *   out : [n_rot][P][m][m][m] float32 (x fastest), host or device. */
dock_status dock_voxelize(dock_ctx* ctx, const dock_probe_desc* probe, const double* rot, int n_rot,
                          float* out);

/* Tuning / introspection ------------------------------------------------------------- */
typedef enum {
    DOCK_TUNE_REGIONS = 1,        /* translation regions per rotation batch (0 = auto; > 0 also turns off
                                     the tcgen05 variant-1 dynamic tile scheduler) */
    DOCK_TUNE_FORCE_FALLBACK = 2, /* 1 => every rotation takes the exact full-grid fallback (tests) */
    DOCK_TUNE_CAND_CAP = 3,       /* candidates kept per rotation before overflow fallback (>= 32) */
    DOCK_TUNE_ENGINE = 4,         /* correlation engine: 0 auto (tcgen05 when eligible), 1 FP32 FFMA, 2 tcgen05,
                                     3 FFT (cuFFT R2C/C2R + this library's channel multiply-accumulate and exact
                                     greedy on the score grids; the paper's FFT method P:L156-163, kept as the
                                     comparison point of the direct-vs-FFT crossover P:L485-502; never auto),
                                     4 sparse ligand (FP32 direct correlation over the occupied probe voxels only:
                                     per-probe atom grids G_a = sum_p w_p coef_ap R_p gathered at each atom's voxel,
                                     P:L504-509, L553-555; needs <= 32 atoms per probe; auto picks it by a cost
                                     model) */
    DOCK_TUNE_TC_VARIANT = 5,     /* tcgen05 kernel: 0 auto, 1 = resident receptor boxes (one channel group, P <= 4,
                                     128 translations x 4 rows per tile), 2 = receptor streamed one (channel group,
                                     z-plane) unit at a time (any P <= 32, m <= 8; 64 / 128 / 160 translations per
                                     row, chosen at init for nx).  A variant that cannot run m falls back to the
                                     other one. */
    DOCK_TUNE_TC_EPILOGUE_WARPS = 6, /* tcgen05 epilogue warps: 0 auto (= the compiled maximum, 8), 4 or 8 (values
                                     above the compiled maximum are clamped to it) */
    DOCK_TUNE_TC_CHUNK = 7,       /* tcgen05 variant 1: tiles per dynamically scheduled chunk (0 = auto, 4..16 by launch length;
                                     1..4096); one persistent CTA per SM takes chunks from a device counter */
    DOCK_TUNE_TC_SCHEDULE = 8,    /* tcgen05 variant 1 schedule.  A ring stage (4 K-steps of 16 products per accumulator)
                                     whose probe weights are zero for all 128 rotations of a block adds exact zeros, so a
                                     block runs only its active stages (a probe grid has at most one occupied voxel per
                                     atom).  0 (default): occupancy schedule, the units first grouped into
                                     blocks with few distinct active stages (greedy, on the device, deterministic); 1:
                                     occupancy schedule over blocks of consecutive units; 2: dense (every stage).  Scores
                                     are bitwise identical in all three modes (skipped products are exact zeros). */
    DOCK_TUNE_SHARD = 9           /* block sharding for multi-GPU runs: value = world << 16 | rank (world 1 = off).  With
                                     world > 1, dock_probe_batch docks only the rotation blocks rank, rank + world, ...
                                     of the call's (clustered, deterministic) block order -- every rank clusters the
                                     whole unit range, so the blocks stay as good as on one GPU -- and writes only its
                                     units' rows of `out` (a DEVICE buffer: host output copies every row back); the caller
                                     pre-fills `out` with 0x80000000 in every field and
                                     combines the ranks' buffers with an elementwise int32 MAX (every field of a written
                                     row is > INT32_MIN except the bits of a -0.0 score, which MAX keeps).  Needs the
                                     tcgen05 variant-1 engine (DOCK_E_UNSUPPORTED otherwise). */
} dock_tune_key;

dock_status dock_set_tuning(dock_ctx* ctx, int key, int64_t value);

typedef struct {
    int lanes_x, tile_x, tile_y, tile_z, n_tiles, n_stages, smem_bytes;
    int regions_last;          /* regions per rotation batch of the last dock_probe_batch (0: tcgen05 variant 1's
                                  dynamic tile scheduler, DOCK_TUNE_TC_CHUNK) */
    int64_t items_last;        /* CTAs launched by the last call's correlation */
    int64_t fallback_last;     /* rotations that took the exact fallback in the last call (valid after its sync point) */
    int64_t cand_max_last;     /* largest candidate count of one rotation in the last call (idem) */
    int64_t kernels_last;      /* kernels launched by the last call */
    int rot_batch;             /* rotations per register block (RB) */
    int x_per_thread;          /* translations along x per thread (XT) */
    int padded_x, padded_y, padded_z;
    double l2_bytes;           /* device L2 size (cudaDevAttrL2CacheSize) */
    double corr_ms_last;       /* CUDA-event duration of the last k_corr launch (dock_probe_batch), -1 if none */
    int n_sms;                 /* multiprocessors of the context's device */
    int engine_last;           /* engine of the last correlation: 1 FP32 FFMA, 2 tcgen05 bf16x3, 3 FFT, 4 sparse */
    int tc_available;          /* 1 if the tcgen05 engine is available for m_max */
    int tc_variant_last;       /* tcgen05 variant of the last correlation (1 or 2), 0 if FFMA */
    int tc_ksteps_last;        /* K-steps (K = 16 each) per translation row executed by the last tcgen05 launch */
    int tc_row_last;           /* translations per MMA row (MMA N) of the last tcgen05 launch */
    int tc_rows_per_tile_last; /* translation rows per tile (TMEM accumulators) of the last tcgen05 launch */
    int pending;               /* 1 if the last asynchronous call has not reached a sync point (dock_sync) */
    int fb_chunk;              /* flagged rotations per iteration of the device-driven fallback loop */
    int sp_atom_grids_last;    /* sparse engine: atom grids G_a computed by the last call */
    int sp_row_last;           /* sparse engine: translations per column row (32 x per-lane count) */
    double sp_terms_last;      /* sparse engine: atoms summed over the units of the last call (gathers per translation) */
    int sp_zt_last;            /* sparse engine: z planes per warp and step of the last call (1 or 2) */
    double tc_ksteps_exec_last; /* tcgen05 variant 1: K-steps per translation row executed by the last call, averaged
                                  over its rotation blocks (occupancy schedule); -1 if none or not yet synced */
} dock_info;

dock_status dock_get_info(const dock_ctx* ctx, dock_info* info);

void dock_destroy(dock_ctx* ctx);
const char* dock_status_string(dock_status s);
const char* dock_last_error(const dock_ctx* ctx);   /* context-local message of the last failure */

#ifdef __cplusplus
}
#endif
#endif /* B200_DOCK_H */

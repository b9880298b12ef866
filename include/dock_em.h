/*
 * dock_em.h -- C ABI of the energy-minimisation non-bonded kernels (libdock.so).
 *
 * Method: Sukhwani & Herbordt, "Fast Binding Site Mapping using GPUs and CUDA", IPPS 2010, §II.B and §IV
 * ("P:L<a>-<b>" cites PAPER.md).  Energy minimisation spends >99 % of its energy evaluation in the
 * non-bonded terms: ACE electrostatics = self energies (Eqs. 4-6) + generalized-
 * Born pair energies (Eq. 7), and a cut-off 6-12 van der Waals variant (Eqs. 8-10,
 * P:L353-470).  The paper maps them onto three GPU kernels -- (a) self energies, (b) pairwise GB + vdW,
 * (c) force updates -- over a pairs list whose per-atom accumulation follows a static
 * assignment table.  Here the pairs list (i < j, sorted by (i, j)) is split at init into
 * the forward segments (pairs whose first atom is a) and the reverse segments (pairs whose second atom
 * is a); every per-atom sum runs over its two segments in a fixed order (deterministic, no atomics).
 *
 * Eqs. 5-8 are garbled in PAPER.md; the readings E1-E6 are those of oracle/em_oracle.c:
 *   tau = 1 - 1/eps_s;  s_i = 1/(2 eps_s R_i) + sum_{k in N(i)} s_ik,
 *   s_ik = tau [omega_ik exp(-r^2/sigma_ik^2) + V_k/(8 pi) (r^3/(r^4 + mu_ik^4))^4]   (type pair (t_i, t_k)),
 *   E_self = 332 sum_i q_i^2 s_i;  Born radius alpha_i = tau / (2 s_i);
 *   E_GB   = sum_pairs 332 q_i q_j (1/r - tau / sqrt(r^2 + a exp(-r^2/(4a)))),  a = alpha_i alpha_j;
 *   E_vdw  = sum_pairs eps_ij [rm^12 (r^-12 + 2 r^6/rc^18 - 3/rc^12) - 2 rm^6 (r^-6 + r^6/rc^12 - 2/rc^6)]
 *            for r < rc (eps_ij = sqrt(eps_i eps_j), rm = (rm_i + rm_j)/2), 0 beyond;
 *   forces = -grad(E_self + E_GB + E_vdw), chain rule through the Born radii included.
 * Arithmetic is FP64 (the paper states no precision; minimisation compares totals of ~1e3-1e4 to
 * ~1e-3, beyond FP32 accumulation).
 * Status codes and conventions are those of dock.h (host or device pointers, one stream per context,
 * calls synchronise before returning).
 */
#ifndef B200_DOCK_EM_H
#define B200_DOCK_EM_H

#include "dock.h"

#ifdef __cplusplus
extern "C" {
#endif

typedef struct dock_em_ctx dock_em_ctx;

typedef struct {
    int n_atoms;     /* >= 1 */
    int n_pairs;     /* >= 0 */
    int n_types;     /* >= 1 */
    int device;      /* CUDA device ordinal */
    double eps_s;    /* solvent dielectric (> 1) */
    double rc;       /* van der Waals cut-off (A, > 0) */
    void* stream;    /* cudaStream_t (cudaStreamLegacy allowed); NULL => the context creates its own */
} dock_em_desc;

typedef struct {     /* host or device pointers; copied by dock_em_init */
    const double *q, *R, *V, *eps, *rm;   /* [n_atoms] charge, intrinsic radius (> 0), volume, vdW eps (>= 0), rm */
    const int* type;                      /* [n_atoms] in [0, n_types) */
    const double *omega, *sigma, *mu;     /* [n_types][n_types], ordered type pair (t_i, t_k); sigma, mu > 0 */
    const int* pairs;                     /* [n_pairs][2]: 0 <= i < j < n_atoms, sorted by (i, j), no duplicates */
} dock_em_params;

/* dock_em_init -- validate and copy the system, build the forward/reverse segment tables. */
dock_status dock_em_init(const dock_em_desc* d, const dock_em_params* p, dock_em_ctx** out);

/* dock_em_eval -- energies and forces of n_conf conformations of the system.
 *   xyz      : [n_conf][n_atoms][3] float64 (A), host or device; must be finite, no two paired atoms coincident.
 *   energies : [n_conf][3] float64 (E_self, E_GB, E_vdw), host or device.
 *   forces   : [n_conf][n_atoms][3] float64 or NULL, host or device. */
dock_status dock_em_eval(dock_em_ctx* ctx, const double* xyz, int n_conf, double* energies, double* forces);

/* Duration (ms, CUDA events) of the kernels of the last dock_em_eval, -1 if none. */
double dock_em_last_ms(const dock_em_ctx* ctx);

void dock_em_destroy(dock_em_ctx* ctx);
const char* dock_em_last_error(const dock_em_ctx* ctx);

#ifdef __cplusplus
}
#endif
#endif /* B200_DOCK_EM_H */

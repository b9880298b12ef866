/*
 * em_oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * Plain FP64 CPU implementation of the non-bonded energy evaluation of FTMap's energy minimisation
 * (Sukhwani & Herbordt, IPPS 2010, §II.B and §IV).  "P:L<a>-<b>" cites PAPER.md.
 * Only tests/ (and bench scripts' reference legs) load this library; it shares no code with csrc/.
 *
 * The non-bonded energy is electrostatics + van der Waals (Eq. 3; >99 % of the energy
 * evaluation).  Eqs. 5-8 are garbled in PAPER.md; the readings (E1-E6) are:
 *   tau = 1 - 1/eps_s (eps_in = 1).
 *   ACE self energy (Eq. 5):   E_i^self = q_i^2 s_i,
 *        s_i = 1/(2 eps_s R_i) + sum_{k in N(i)} s_ik                               (reading E1)
 *   pairwise self term (Eq. 6): s_ik = tau [ omega_ik exp(-r^2/sigma_ik^2)
 *                                                 + Vt_k/(8 pi) (r^3/(r^4 + mu_ik^4))^4 ]   (reading E2)
 *        (omega, sigma, mu indexed by the ordered type pair (type_i, type_k); Vt_k the volume of atom k)
 *   Born radius ("depend on the self-energy"): alpha_i = tau / (2 s_i)      (reading E3)
 *   GB pair energy (Eq. 7):  E_ij = 332 q_i q_j / r - 332 tau q_i q_j / f_ij,
 *        f_ij = sqrt(r^2 + a exp(-r^2/(4 a))), a = alpha_i alpha_j                      (reading E4)
 *   vdW (Eqs. 8-10): eps_ij = sqrt(eps_i eps_j), rm_ij = (rm_i + rm_j)/2, shifted 6-12:
 *        E = eps_ij [ rm^12 (r^-12 + 2 r^6/rc^18 - 3/rc^12) - 2 rm^6 (r^-6 + r^6/rc^12 - 2/rc^6) ] for r < rc,
 *        0 beyond (E(rc) = E'(rc) = 0)                                                   (reading E5)
 *   Totals: E_self = 332 sum_i E_i^self, E_GB = sum_pairs E_ij, E_vdw = sum_pairs E_ij^vdw.
 *   Forces F = -grad(E_self + E_GB + E_vdw), with the chain rule through the Born radii.  (reading E6)
 * N(i) = the partners of i in the pair list (pairs i < j given once, used for both atoms).
 *
 * Every function here is pinned by tests/test_em_oracle_pins.py (finite-difference gradients, Newton's
 * third law, rigid-motion and label-permutation invariance, closed forms of the limits).
 */
#include <math.h>
#include <stdlib.h>
#include <string.h>

#ifdef _OPENMP
#include <omp.h>
#endif

#define EM_PI 3.14159265358979323846

typedef struct {
    int n_atoms, n_pairs, n_types;
    const double *q, *R, *V, *eps, *rm;   /* [n_atoms] */
    const int* type;                       /* [n_atoms] */
    const double *omega, *sigma, *mu;      /* [n_types][n_types], ordered pair (type_i, type_k) */
    const int* pairs;                      /* [n_pairs][2], i < j */
    double eps_s, rc;
} em_sys;

/* s_ik and d s_ik / dr for the ordered pair (i <- k): Eq. 6 reading E2. */
static void self_term(const em_sys* S, int i, int k, double r, double* s, double* ds)
{
    const double tau = 1.0 - 1.0 / S->eps_s;
    const int t = S->type[i] * S->n_types + S->type[k];
    const double om = S->omega[t], sg = S->sigma[t], mu = S->mu[t];
    const double ga = exp(-r * r / (sg * sg));
    const double d = r * r * r * r + mu * mu * mu * mu;
    const double g = r * r * r / d;
    const double dg = (3.0 * r * r * d - r * r * r * 4.0 * r * r * r) / (d * d);
    *s = tau * (om * ga + S->V[k] / (8.0 * EM_PI) * g * g * g * g);
    *ds = tau * (om * ga * (-2.0 * r / (sg * sg)) + S->V[k] / (8.0 * EM_PI) * 4.0 * g * g * g * dg);
}

/* One conformation x [n_atoms][3] -> e[3] = (E_self, E_GB, E_vdw) and, if f != NULL, forces f[n_atoms][3]. */
void orc_em_eval(const em_sys* S, const double* x, double* e, double* f)
{
    const int n = S->n_atoms, np = S->n_pairs;
    const double tau = 1.0 - 1.0 / S->eps_s, rc = S->rc;
    double* s = (double*)calloc(n, sizeof(double));
    double* G = (double*)calloc(n, sizeof(double));     /* sum_j dE_GB/dalpha_i */
    double* alpha = (double*)calloc(n, sizeof(double));
    double e_self = 0.0, e_gb = 0.0, e_vdw = 0.0;
    for (int i = 0; i < n; i++) s[i] = 1.0 / (2.0 * S->eps_s * S->R[i]);
    for (int p = 0; p < np; p++) {   /* Eq. 5: sum of the pairwise self terms over the neighbours */
        const int i = S->pairs[2 * p], j = S->pairs[2 * p + 1];
        const double dx = x[3 * i] - x[3 * j], dy = x[3 * i + 1] - x[3 * j + 1], dz = x[3 * i + 2] - x[3 * j + 2];
        const double r = sqrt(dx * dx + dy * dy + dz * dz);
        double sij, dsij, sji, dsji;
        self_term(S, i, j, r, &sij, &dsij);
        self_term(S, j, i, r, &sji, &dsji);
        s[i] += sij;
        s[j] += sji;
    }
    for (int i = 0; i < n; i++) {
        e_self += 332.0 * S->q[i] * S->q[i] * s[i];
        alpha[i] = tau / (2.0 * s[i]);   /* reading E3 */
    }
    if (f) memset(f, 0, sizeof(double) * 3 * n);
    /* pairwise GB + vdW, and dE_GB/dalpha */
    double* dEdr = (double*)calloc(np > 0 ? np : 1, sizeof(double));
    for (int p = 0; p < np; p++) {
        const int i = S->pairs[2 * p], j = S->pairs[2 * p + 1];
        const double dx = x[3 * i] - x[3 * j], dy = x[3 * i + 1] - x[3 * j + 1], dz = x[3 * i + 2] - x[3 * j + 2];
        const double r = sqrt(dx * dx + dy * dy + dz * dz);
        const double qq = S->q[i] * S->q[j];
        const double a = alpha[i] * alpha[j];
        const double ex = exp(-r * r / (4.0 * a));
        const double f2 = r * r + a * ex;
        const double fg = sqrt(f2);
        e_gb += 332.0 * qq / r - 332.0 * tau * qq / fg;
        const double df2dr = 2.0 * r - 0.5 * r * ex;
        const double df2da = ex * (1.0 + r * r / (4.0 * a));
        const double dEdf2 = 332.0 * tau * qq * 0.5 / (f2 * fg);   /* d(-332 tau qq f^-1)/d(f^2) */
        G[i] += dEdf2 * df2da * alpha[j];
        G[j] += dEdf2 * df2da * alpha[i];
        double de = -332.0 * qq / (r * r) + dEdf2 * df2dr;
        if (r < rc) {   /* Eqs. 8-10, reading E5 */
            const double eps = sqrt(S->eps[i] * S->eps[j]), rm = 0.5 * (S->rm[i] + S->rm[j]);
            const double rm6 = rm * rm * rm * rm * rm * rm, rm12 = rm6 * rm6;
            const double r2 = r * r, r6 = r2 * r2 * r2, rc6 = rc * rc * rc * rc * rc * rc;
            e_vdw += eps * (rm12 * (1.0 / (r6 * r6) + 2.0 * r6 / (rc6 * rc6 * rc6) - 3.0 / (rc6 * rc6)) -
                            2.0 * rm6 * (1.0 / r6 + r6 / (rc6 * rc6) - 2.0 / rc6));
            de += eps * (rm12 * (-12.0 / (r6 * r6 * r) + 12.0 * r6 / (r * rc6 * rc6 * rc6)) -
                         2.0 * rm6 * (-6.0 / (r6 * r) + 6.0 * r6 / (r * rc6 * rc6)));
        }
        dEdr[p] = de;
    }
    if (f) {
        /* chain rule through the self energies: c_i = dE/ds_i = 332 q_i^2 + G_i dalpha_i/ds_i */
        for (int p = 0; p < np; p++) {
            const int i = S->pairs[2 * p], j = S->pairs[2 * p + 1];
            const double dx = x[3 * i] - x[3 * j], dy = x[3 * i + 1] - x[3 * j + 1], dz = x[3 * i + 2] - x[3 * j + 2];
            const double r = sqrt(dx * dx + dy * dy + dz * dz);
            double sij, dsij, sji, dsji;
            self_term(S, i, j, r, &sij, &dsij);
            self_term(S, j, i, r, &sji, &dsji);
            const double ci = 332.0 * S->q[i] * S->q[i] + G[i] * (-tau / (2.0 * s[i] * s[i]));
            const double cj = 332.0 * S->q[j] * S->q[j] + G[j] * (-tau / (2.0 * s[j] * s[j]));
            const double de = dEdr[p] + ci * dsij + cj * dsji;
            const double ux = dx / r, uy = dy / r, uz = dz / r;
            f[3 * i] -= de * ux;
            f[3 * i + 1] -= de * uy;
            f[3 * i + 2] -= de * uz;
            f[3 * j] += de * ux;
            f[3 * j + 1] += de * uy;
            f[3 * j + 2] += de * uz;
        }
    }
    e[0] = e_self;
    e[1] = e_gb;
    e[2] = e_vdw;
    free(s);
    free(G);
    free(alpha);
    free(dEdr);
}

/* Many conformations: x [n_conf][n_atoms][3] -> e [n_conf][3], f [n_conf][n_atoms][3] (may be NULL). */
void orc_em_eval_batch(const em_sys* S, int n_conf, const double* x, double* e, double* f, int n_threads)
{
#ifdef _OPENMP
    if (n_threads > 0) omp_set_num_threads(n_threads);
#else
    (void)n_threads;
#endif
#pragma omp parallel for schedule(dynamic, 1)
    for (int c = 0; c < n_conf; c++)
        orc_em_eval(S, x + (size_t)3 * S->n_atoms * c, e + 3 * (size_t)c,
                    f ? f + (size_t)3 * S->n_atoms * c : NULL);
}

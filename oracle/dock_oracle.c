/*
 * dock_oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * A plain, slow, obviously-correct FP64 CPU implementation of the rigid-docking
 * hot path of Sukhwani & Herbordt, "Fast Binding Site Mapping using GPUs and
 * CUDA" (IPPS/IPDPS 2010).  Citations "P:L<a>-<b>" point into PAPER.md.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline/reference
 * leg may load this library.  It shares no code, header, table or constant
 * with the CUDA path (paper_conf_ipps_sukhwanih10_b200/csrc); neither side
 * includes or links the other.
 *
 * What it computes (readings Q1-Q22 listed in DESIGN.md):
 *   1. voxelize  -- grid assignment of the rotated probe:
 *        g = (Q x)/h + c, c = (m-1)/2;  v = floor(g + 0.5) per axis;
 *        L_p[v] += coef[a][p]; an atom outside [0,m)^3 is an error (reading Q3).
 *   2. score     -- Eq. 1 + Eq. 2, direct correlation
 *        "sum of all the voxel-voxel interactions for each translation"
 *        (P:L504-509):  S[t] = sum_p w_p sum_v L_p[v] R_p[(t+v) mod n]
 *        (cyclic, reading Q1/Q2), plus A[t] = sum_p sum_v |w_p L_p[v] R_p[.]|
 *        for the tolerance (reading Q16).
 *   3. filter    -- "selecting the best score and then excluding its neighbors
 *        while selecting the next best score" (Fig. 5),
 *        with the exclusion array of length N^3: k times pick the
 *        minimum (score, t_lin) among available cells, then mark every cell
 *        within cyclic Chebyshev distance rho unavailable (readings Q7-Q9).
 *        k = 4 per rotation in FTMap.
 *   4. dock      -- 1-3 for every (probe, rotation) unit, OpenMP over units.
 *
 * Parity pins for every function live in tests/test_oracle_pins.py (A, the tolerance scale of
 * every GPU parity check, is pinned by P13).
 */
#include <math.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

#ifdef _OPENMP
#include <omp.h>
#endif

#define ORC_OK 0
#define ORC_E_INVALID (-1)
#define ORC_E_OUTSIDE (-3)
#define ORC_E_BAD_ROTATION (-4)

/* |Q^T Q - I| <= 1e-9 elementwise and det(Q) > 0  (reading Q5: caller supplies proper rotations). */
int orc_check_rotation(const double* q)
{
    for (int i = 0; i < 3; i++)
        for (int j = 0; j < 3; j++) {
            double s = 0.0;
            for (int l = 0; l < 3; l++) s += q[3 * l + i] * q[3 * l + j];
            double want = (i == j) ? 1.0 : 0.0;
            if (!(fabs(s - want) <= 1e-9)) return ORC_E_BAD_ROTATION;
        }
    double det = q[0] * (q[4] * q[8] - q[5] * q[7])
               - q[1] * (q[3] * q[8] - q[5] * q[6])
               + q[2] * (q[3] * q[7] - q[4] * q[6]);
    return det > 0.0 ? ORC_OK : ORC_E_BAD_ROTATION;
}

/* Step 1: voxelize one rotated probe.  L is [P][m][m][m] (x fastest), zeroed here. */
int orc_voxelize(const double* xyz, const float* coef, int n_atoms, int P, int m,
                 const double* q, double spacing, double* L)
{
    if (m < 1 || P < 1 || n_atoms < 0 || !(spacing > 0.0)) return ORC_E_INVALID;
    memset(L, 0, sizeof(double) * (size_t)P * m * m * m);
    double c = (m - 1) / 2.0;
    for (int a = 0; a < n_atoms; a++) {
        const double* x = xyz + 3 * a;
        int v[3];
        for (int i = 0; i < 3; i++) {
            double rx = q[3 * i + 0] * x[0] + q[3 * i + 1] * x[1] + q[3 * i + 2] * x[2];
            double g = rx / spacing + c;
            double f = floor(g + 0.5);
            if (!(f >= 0.0 && f < (double)m)) return ORC_E_OUTSIDE;
            v[i] = (int)f;
        }
        for (int p = 0; p < P; p++)
            L[(((size_t)p * m + v[2]) * m + v[1]) * m + v[0]] += (double)coef[(size_t)a * P + p];
    }
    return ORC_OK;
}

/* Step 2: score grid S (and magnitude sum A, may be NULL) for one voxelized probe.
 * R is [P][nz][ny][nx] float32, L is [P][m][m][m] double, w is [P] float32.
 * S[t] = sum_p w_p sum_{v in [0,m)^3} L_p[v] * R_p[(t+v) mod n],  t_lin = (tz*ny + ty)*nx + tx. */
void orc_score_grid(const float* R, int nx, int ny, int nz, int P, const double* L, int m,
                    const float* w, double* S, double* A)
{
    for (int tz = 0; tz < nz; tz++)
        for (int ty = 0; ty < ny; ty++)
            for (int tx = 0; tx < nx; tx++) {
                double s = 0.0, a = 0.0;
                for (int p = 0; p < P; p++)
                    for (int vz = 0; vz < m; vz++)
                        for (int vy = 0; vy < m; vy++)
                            for (int vx = 0; vx < m; vx++) {
                                double l = L[(((size_t)p * m + vz) * m + vy) * m + vx];
                                int z = (tz + vz) % nz, y = (ty + vy) % ny, x = (tx + vx) % nx;
                                double r = (double)R[(((size_t)p * nz + z) * ny + y) * nx + x];
                                double term = (double)w[p] * l * r;
                                s += term;
                                a += fabs(term);
                            }
                size_t t = ((size_t)tz * ny + ty) * nx + tx;
                S[t] = s;
                if (A) A[t] = a;
            }
}

/* Step 3: greedy filter with an N^3 exclusion array.
 * Picks k cells in order; ties in score are broken by the smaller t_lin (reading Q8;
 * -0.0 == +0.0 holds for doubles).  Returns the number of picks made (< k only when
 * every cell has been excluded). */
int orc_filter(const double* S, int nx, int ny, int nz, int k, int rho, int64_t* t_out, double* s_out)
{
    size_t n = (size_t)nx * ny * nz;
    unsigned char* excluded = (unsigned char*)calloc(n, 1);
    if (!excluded) return ORC_E_INVALID;
    int picks = 0;
    for (int j = 0; j < k; j++) {
        size_t best = n;
        for (size_t t = 0; t < n; t++) {
            if (excluded[t]) continue;
            if (best == n || S[t] < S[best]) best = t;   /* strict <: earlier (smaller) t_lin wins ties */
        }
        if (best == n) break;
        t_out[j] = (int64_t)best;
        s_out[j] = S[best];
        picks++;
        int bx = (int)(best % nx), by = (int)((best / nx) % ny), bz = (int)(best / ((size_t)nx * ny));
        for (int dz = -rho; dz <= rho; dz++)
            for (int dy = -rho; dy <= rho; dy++)
                for (int dx = -rho; dx <= rho; dx++) {
                    int x = ((bx + dx) % nx + nx) % nx;
                    int y = ((by + dy) % ny + ny) % ny;
                    int z = ((bz + dz) % nz + nz) % nz;
                    excluded[((size_t)z * ny + y) * nx + x] = 1;
                }
    }
    free(excluded);
    return picks;
}

/* Step 4: full rigid docking over (probe, rotation) units [unit_begin, unit_end),
 * units ordered probe-major (unit = probe * n_rot + rotation).
 *   probes: xyz_all/coef_all concatenated, atom_off[n_probes+1], m per probe.
 *   out_t  [n_units][k] int64 (-1 when fewer picks), out_s [n_units][k] double,
 *   out_a  [n_units][k] double or NULL: the magnitude sum A (reading Q16) at each pick,
 *          the tolerance scale a GPU score is compared with,
 *   out_status [n_units] int (0 or an ORC_E_* code).
 * Uses OpenMP over units when compiled with -fopenmp; n_threads <= 0 => library default. */
int orc_dock(const float* R, int nx, int ny, int nz, int P, const float* w, double spacing,
             const double* xyz_all, const float* coef_all, const int* atom_off, const int* m_of,
             int n_probes, const double* rot, int n_rot, int64_t unit_begin, int64_t unit_end,
             int k, int rho, int n_threads, int64_t* out_t, double* out_s, double* out_a,
             int* out_status)
{
    if (unit_begin < 0 || unit_end < unit_begin || unit_end > (int64_t)n_probes * n_rot || k < 1)
        return ORC_E_INVALID;
    int64_t n_units = unit_end - unit_begin;
    size_t ncell = (size_t)nx * ny * nz;
#ifdef _OPENMP
    if (n_threads > 0) omp_set_num_threads(n_threads);
#else
    (void)n_threads;
#endif
    int m_big = 1;
    for (int pr = 0; pr < n_probes; pr++) if (m_of[pr] > m_big) m_big = m_of[pr];
#pragma omp parallel
    {
        double* S = (double*)malloc(sizeof(double) * ncell);
        double* A = out_a ? (double*)malloc(sizeof(double) * ncell) : NULL;
        double* L = (double*)malloc(sizeof(double) * (size_t)P * m_big * m_big * m_big);
#pragma omp for schedule(dynamic, 1)
        for (int64_t i = 0; i < n_units; i++) {
            int64_t u = unit_begin + i;
            int pr = (int)(u / n_rot), r = (int)(u % n_rot);
            int m = m_of[pr];
            for (int j = 0; j < k; j++) {
                out_t[i * k + j] = -1;
                out_s[i * k + j] = NAN;
                if (out_a) out_a[i * k + j] = NAN;
            }
            int st = orc_check_rotation(rot + 9 * (size_t)r);
            if (st == ORC_OK)
                st = orc_voxelize(xyz_all + 3 * (size_t)atom_off[pr], coef_all + (size_t)P * atom_off[pr],
                                  atom_off[pr + 1] - atom_off[pr], P, m, rot + 9 * (size_t)r, spacing, L);
            out_status[i] = st;
            if (st != ORC_OK) continue;
            orc_score_grid(R, nx, ny, nz, P, L, m, w, S, A);
            int np = orc_filter(S, nx, ny, nz, k, rho, out_t + i * k, out_s + i * k);
            if (out_a)
                for (int j = 0; j < np; j++) out_a[i * k + j] = A[out_t[i * k + j]];
        }
        free(S);
        free(A);
        free(L);
    }
    return ORC_OK;
}

int orc_max_threads(void)
{
#ifdef _OPENMP
    return omp_get_max_threads();
#else
    return 1;
#endif
}

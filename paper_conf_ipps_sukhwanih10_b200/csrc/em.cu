// em.cu -- energy-minimisation non-bonded kernels (include/dock_em.h).
//
// The paper's three GPU kernels: (a) self energies, (b) pairwise GB + vdW, (c) force update,
// over a pairs list accumulated per atom through a static assignment table.  Here:
//   k_em_self   (a)  per (conformation, atom): s_a over its forward + reverse pair segments -> Born radius
//   k_em_pair   (b)  per (conformation, pair): GB + vdW energies, dE/dr at fixed radii, dE/dalpha_i,j
//   k_em_chain       per (conformation, atom): c_a = dE/ds_a (self energy + GB through the Born radius)
//   k_em_force  (c)  per (conformation, atom): F_a from its segments (pair terms + chain-rule terms; the
//                    self-term derivatives of both sides come from k_em_self, which evaluates each once)
//   k_em_energy      per conformation: the three totals (fixed-order block reduction)
// The split forward/reverse pairs lists of P:L799-881 are the two segment tables built at init; every
// per-atom accumulation is one warp over the atom's segments (lane-strided, then a fixed xor tree):
// deterministic, no atomics.  FP64.
#include <cuda_runtime.h>

#include <algorithm>
#include <cmath>
#include <cstdarg>
#include <cstdio>
#include <cstring>
#include <new>
#include <vector>

#include "dock_em.h"

namespace em {

constexpr double PI = 3.14159265358979323846;

struct Sys {
    int n, np, T;
    double eps_s, rc, tau;
    const double *q, *R, *V, *eps, *rm;
    const int* type;
    const double *omega, *sigma, *mu;
    const int2* pairs;      // [np] (i, j), i < j, sorted
    const int* fwd_off;     // [n + 1]: pairs of atom a as first atom: [fwd_off[a], fwd_off[a+1])
    const int* rev_off;     // [n + 1]: rev_pair[rev_off[a] .. rev_off[a+1]) = pairs with a as second atom
    const int* rev_pair;    // [np]
};

// s_ik and ds_ik/dr for the ordered pair (i <- k) (Eq. 6, reading E2)
__device__ __forceinline__ void self_term(const Sys& S, int i, int k, double r, double& s, double& ds)
{
    const int t = S.type[i] * S.T + S.type[k];
    const double om = S.omega[t], sg = S.sigma[t], mu = S.mu[t];
    const double ga = exp(-r * r / (sg * sg));
    const double mu4 = mu * mu * mu * mu;
    const double r2 = r * r, r3 = r2 * r;
    const double d = r2 * r2 + mu4;
    const double g = r3 / d;
    const double dg = (3.0 * r2 * d - r3 * 4.0 * r3) / (d * d);
    const double g3 = g * g * g;
    const double vk = S.V[k] / (8.0 * PI);
    s = S.tau * (om * ga + vk * g3 * g);
    ds = S.tau * (om * ga * (-2.0 * r / (sg * sg)) + vk * 4.0 * g3 * dg);
}

__device__ __forceinline__ double dist(const double* xc, int a, int b, double& dx, double& dy, double& dz)
{
    dx = xc[3 * a] - xc[3 * b];
    dy = xc[3 * a + 1] - xc[3 * b + 1];
    dz = xc[3 * a + 2] - xc[3 * b + 2];
    return sqrt(dx * dx + dy * dy + dz * dz);
}

// One warp per (conformation, atom): lane l takes the atom's neighbours l, l + 32, ... of its forward then
// reverse segment, and the lane partial sums are combined by a fixed xor tree -- deterministic, independent of
// the batch, 32 gathers in flight per atom.
__device__ __forceinline__ double warp_sum(double v)
{
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(0xffffffffu, v, o);
    return v;
}
// neighbour j of atom a (forward segment first): pair index and partner atom
__device__ __forceinline__ void neighbour(const Sys& S, int a, int nf, int j, int& p, int& k)
{
    if (j < nf) {
        p = S.fwd_off[a] + j;
        k = S.pairs[p].y;
    } else {
        p = S.rev_pair[S.rev_off[a] + j - nf];
        k = S.pairs[p].x;
    }
}

// (a) self energies: s_a = 1/(2 eps_s R_a) + sum over a's neighbours (Eq. 5), Born radius (reading E3)
__global__ void k_em_self(Sys S, const double* __restrict__ x, int nconf, double* s_out, double* alpha_out,
                          double* eself, double2* dsd)
{
    const long long w = (blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x) >> 5;
    const int lane = threadIdx.x & 31;
    if (w >= static_cast<long long>(nconf) * S.n) return;   // warp-uniform
    const int c = static_cast<int>(w / S.n), a = static_cast<int>(w % S.n);
    const double* xc = x + static_cast<size_t>(c) * S.n * 3;
    const int nf = S.fwd_off[a + 1] - S.fwd_off[a], nn = nf + S.rev_off[a + 1] - S.rev_off[a];
    double s = 0.0, dx, dy, dz, t, dt;
    double* ds_out = reinterpret_cast<double*>(dsd + static_cast<size_t>(c) * S.np);
    for (int j = lane; j < nn; j += 32) {
        int p, k;
        neighbour(S, a, nf, j, p, k);
        self_term(S, a, k, dist(xc, a, k, dx, dy, dz), t, dt);
        s += t;
        ds_out[2 * static_cast<size_t>(p) + (j < nf ? 0 : 1)] = dt;   // ds_ak/dr for the force pass (this side)
    }
    s = warp_sum(s) + 1.0 / (2.0 * S.eps_s * S.R[a]);
    if (lane == 0) {
        s_out[w] = s;
        alpha_out[w] = S.tau / (2.0 * s);
        eself[w] = 332.0 * S.q[a] * S.q[a] * s;
    }
}

// (b) pairwise GB (Eq. 7, reading E4) + shifted 6-12 vdW (Eqs. 8-10, reading E5): energies, dE/dr at fixed
// Born radii, dE/dalpha of both atoms
__global__ void k_em_pair(Sys S, const double* __restrict__ x, int nconf, const double* __restrict__ alpha,
                          double2* e_pair, double* dEdr, double2* dal)
{
    const long long idx = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x;
    if (idx >= static_cast<long long>(nconf) * S.np) return;
    const int c = static_cast<int>(idx / S.np), p = static_cast<int>(idx % S.np);
    const double* xc = x + static_cast<size_t>(c) * S.n * 3;
    const int i = S.pairs[p].x, j = S.pairs[p].y;
    double dx, dy, dz;
    const double r = dist(xc, i, j, dx, dy, dz);
    const double ai = alpha[static_cast<size_t>(c) * S.n + i], aj = alpha[static_cast<size_t>(c) * S.n + j];
    const double qq = S.q[i] * S.q[j];
    const double a = ai * aj;
    const double ex = exp(-r * r / (4.0 * a));
    const double f2 = r * r + a * ex;
    const double fg = sqrt(f2);
    const double egb = 332.0 * qq / r - 332.0 * S.tau * qq / fg;
    const double df2dr = 2.0 * r - 0.5 * r * ex;
    const double df2da = ex * (1.0 + r * r / (4.0 * a));
    const double dEdf2 = 332.0 * S.tau * qq * 0.5 / (f2 * fg);
    double de = -332.0 * qq / (r * r) + dEdf2 * df2dr, evdw = 0.0;
    if (r < S.rc) {
        const double eps = sqrt(S.eps[i] * S.eps[j]), rm = 0.5 * (S.rm[i] + S.rm[j]);
        const double rm6 = rm * rm * rm * rm * rm * rm, rm12 = rm6 * rm6;
        const double r2 = r * r, r6 = r2 * r2 * r2, rc = S.rc, rc6 = rc * rc * rc * rc * rc * rc;
        evdw = eps * (rm12 * (1.0 / (r6 * r6) + 2.0 * r6 / (rc6 * rc6 * rc6) - 3.0 / (rc6 * rc6)) -
                      2.0 * rm6 * (1.0 / r6 + r6 / (rc6 * rc6) - 2.0 / rc6));
        de += eps * (rm12 * (-12.0 / (r6 * r6 * r) + 12.0 * r6 / (r * rc6 * rc6 * rc6)) -
                     2.0 * rm6 * (-6.0 / (r6 * r) + 6.0 * r6 / (r * rc6 * rc6)));
    }
    e_pair[idx] = make_double2(egb, evdw);
    dEdr[idx] = de;
    dal[idx] = make_double2(dEdf2 * df2da * aj, dEdf2 * df2da * ai);
}

// c_a = dE/ds_a = 332 q_a^2 + (sum of dE_GB/dalpha_a over a's pairs) * dalpha_a/ds_a (reading E6); warp per atom
__global__ void k_em_chain(Sys S, int nconf, const double* __restrict__ s, const double2* __restrict__ dal,
                           double* cfac)
{
    const long long w = (blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x) >> 5;
    const int lane = threadIdx.x & 31;
    if (w >= static_cast<long long>(nconf) * S.n) return;
    const int c = static_cast<int>(w / S.n), a = static_cast<int>(w % S.n);
    const double2* dc = dal + static_cast<size_t>(c) * S.np;
    const int nf = S.fwd_off[a + 1] - S.fwd_off[a], nn = nf + S.rev_off[a + 1] - S.rev_off[a];
    double G = 0.0;
    for (int j = lane; j < nn; j += 32) {
        int p, k;
        neighbour(S, a, nf, j, p, k);
        G += j < nf ? dc[p].x : dc[p].y;
    }
    G = warp_sum(G);
    if (lane == 0) {
        const double sa = s[w];
        cfac[w] = 332.0 * S.q[a] * S.q[a] + G * (-S.tau / (2.0 * sa * sa));
    }
}

// (c) forces: F_a = -sum over a's pairs of (dE/dr_p + c_a ds_ak/dr + c_k ds_ka/dr) (x_a - x_k)/r; warp per atom
__global__ void k_em_force(Sys S, const double* __restrict__ x, int nconf, const double* __restrict__ dEdr,
                           const double2* __restrict__ dsd, const double* __restrict__ cfac, double* f)
{
    const long long w = (blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x) >> 5;
    const int lane = threadIdx.x & 31;
    if (w >= static_cast<long long>(nconf) * S.n) return;
    const int c = static_cast<int>(w / S.n), a = static_cast<int>(w % S.n);
    const double* xc = x + static_cast<size_t>(c) * S.n * 3;
    const double* dr = dEdr + static_cast<size_t>(c) * S.np;
    const double* cf = cfac + static_cast<size_t>(c) * S.n;
    const double ca = cf[a];
    const int nf = S.fwd_off[a + 1] - S.fwd_off[a], nn = nf + S.rev_off[a + 1] - S.rev_off[a];
    const double2* dsc = dsd + static_cast<size_t>(c) * S.np;
    double fx = 0.0, fy = 0.0, fz = 0.0, dx, dy, dz;
    for (int j = lane; j < nn; j += 32) {
        int p, k;
        neighbour(S, a, nf, j, p, k);
        const double r = dist(xc, a, k, dx, dy, dz);
        const double2 ds = dsc[p];   // (ds_ij/dr, ds_ji/dr) of pair p = (i, j), from k_em_self
        const double dak = j < nf ? ds.x : ds.y, dka = j < nf ? ds.y : ds.x;
        const double de = (dr[p] + ca * dak + cf[k] * dka) / r;
        fx -= de * dx;
        fy -= de * dy;
        fz -= de * dz;
    }
    fx = warp_sum(fx);
    fy = warp_sum(fy);
    fz = warp_sum(fz);
    if (lane == 0) {
        f[3 * w] = fx;
        f[3 * w + 1] = fy;
        f[3 * w + 2] = fz;
    }
}

// per conformation: E_self = sum over atoms, E_GB and E_vdw = sums over pairs (fixed-order reduction)
__global__ void k_em_energy(int n, int np, const double* __restrict__ eself, const double2* __restrict__ e_pair,
                            double* out)
{
    __shared__ double sh[3][256];
    const int c = blockIdx.x, t = threadIdx.x;
    double a = 0.0, b = 0.0, v = 0.0;
    for (int i = t; i < n; i += 256) a += eself[static_cast<size_t>(c) * n + i];
    for (int p = t; p < np; p += 256) {
        const double2 e = e_pair[static_cast<size_t>(c) * np + p];
        b += e.x;
        v += e.y;
    }
    sh[0][t] = a;
    sh[1][t] = b;
    sh[2][t] = v;
    __syncthreads();
    for (int w = 128; w > 0; w >>= 1) {
        if (t < w)
            for (int q = 0; q < 3; q++) sh[q][t] += sh[q][t + w];
        __syncthreads();
    }
    if (t < 3) out[3 * c + t] = sh[t][0];
}

}  // namespace em

struct dock_em_ctx {
    int device = 0;
    cudaStream_t stream = nullptr;
    bool own_stream = false;
    em::Sys S{};
    void* blob = nullptr;          // device copy of every parameter array
    double *s = nullptr, *alpha = nullptr, *eself = nullptr, *dEdr = nullptr, *cfac = nullptr;
    double2 *e_pair = nullptr, *dal = nullptr, *dsd = nullptr;
    double *d_x = nullptr, *d_e = nullptr, *d_f = nullptr;
    int cap_conf = 0;
    cudaEvent_t ev[2] = {nullptr, nullptr};
    bool ev_valid = false;
    bool dead = false;
    char err[256] = {0};
};

namespace {

dock_status em_fail(dock_em_ctx* c, dock_status s, const char* fmt, ...)
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

#define ECU(call)                                                                                             \
    do {                                                                                                      \
        cudaError_t e_ = (call);                                                                              \
        if (e_ != cudaSuccess)                                                                                \
            return em_fail(ctx, e_ == cudaErrorMemoryAllocation ? DOCK_E_OOM : DOCK_E_CUDA, "%s: %s", #call, \
                           cudaGetErrorString(e_));                                                           \
    } while (0)

int em_ptr_kind(const void* p, int device)
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

// copy n elements of a host-or-device array to host
template <typename T>
bool fetch(const T* src, size_t n, std::vector<T>& dst, int device)
{
    dst.resize(n);
    if (!n) return true;
    const int k = em_ptr_kind(src, device);
    if (k < 0) return false;
    if (k == 1) return cudaMemcpy(dst.data(), src, sizeof(T) * n, cudaMemcpyDeviceToHost) == cudaSuccess;
    memcpy(dst.data(), src, sizeof(T) * n);
    return true;
}

void em_free(dock_em_ctx* c)
{
    void* bufs[] = {c->blob, c->s, c->alpha, c->eself, c->dEdr, c->cfac, c->e_pair, c->dal, c->dsd,
                    c->d_x,  c->d_e, c->d_f};
    for (void* b : bufs)
        if (b) cudaFree(b);
    c->s = c->alpha = c->eself = c->dEdr = c->cfac = c->d_x = c->d_e = c->d_f = nullptr;
    c->e_pair = c->dal = c->dsd = nullptr;
    c->blob = nullptr;
}

}  // namespace

extern "C" {

const char* dock_em_last_error(const dock_em_ctx* ctx) { return ctx ? ctx->err : "null context"; }

double dock_em_last_ms(const dock_em_ctx* ctx)
{
    if (!ctx || !ctx->ev_valid) return -1.0;
    float ms = 0.f;
    if (cudaEventElapsedTime(&ms, ctx->ev[0], ctx->ev[1]) != cudaSuccess) {
        cudaGetLastError();
        return -1.0;
    }
    return ms;
}

void dock_em_destroy(dock_em_ctx* ctx)
{
    if (!ctx) return;
    cudaSetDevice(ctx->device);
    if (ctx->stream) cudaStreamSynchronize(ctx->stream);
    em_free(ctx);
    for (cudaEvent_t e : ctx->ev)
        if (e) cudaEventDestroy(e);
    if (ctx->own_stream && ctx->stream) cudaStreamDestroy(ctx->stream);
    cudaGetLastError();
    delete ctx;
}

dock_status dock_em_init(const dock_em_desc* d, const dock_em_params* p, dock_em_ctx** out)
{
    if (!out) return DOCK_E_INVALID_ARG;
    *out = nullptr;
    if (!d || !p) return DOCK_E_INVALID_ARG;
    if (d->n_atoms < 1 || d->n_pairs < 0 || d->n_types < 1 || !(d->eps_s > 1.0) || !(d->rc > 0.0) ||
        !std::isfinite(d->eps_s) || !std::isfinite(d->rc))
        return DOCK_E_INVALID_ARG;
    if ((int64_t)d->n_types * d->n_types > (1 << 20)) return DOCK_E_UNSUPPORTED;
    if (!p->q || !p->R || !p->V || !p->eps || !p->rm || !p->type || !p->omega || !p->sigma || !p->mu ||
        (d->n_pairs > 0 && !p->pairs))
        return DOCK_E_INVALID_ARG;
    dock_em_ctx* ctx = new (std::nothrow) dock_em_ctx();
    if (!ctx) return DOCK_E_OOM;
    auto bail = [&](dock_status s) {
        dock_em_destroy(ctx);
        return s;
    };
    ctx->device = d->device;
    if (cudaSetDevice(d->device) != cudaSuccess) {
        cudaGetLastError();
        return bail(DOCK_E_CUDA);
    }
    if (d->stream) {
        ctx->stream = static_cast<cudaStream_t>(d->stream);
    } else {
        if (cudaStreamCreateWithFlags(&ctx->stream, cudaStreamNonBlocking) != cudaSuccess) return bail(DOCK_E_CUDA);
        ctx->own_stream = true;
    }
    if (cudaEventCreate(&ctx->ev[0]) != cudaSuccess || cudaEventCreate(&ctx->ev[1]) != cudaSuccess)
        return bail(DOCK_E_CUDA);
    const int n = d->n_atoms, np = d->n_pairs, T = d->n_types;
    std::vector<double> q, R, V, eps, rm, om, sg, mu;
    std::vector<int> type, pr;
    const int dev = d->device;
    if (!fetch(p->q, n, q, dev) || !fetch(p->R, n, R, dev) || !fetch(p->V, n, V, dev) ||
        !fetch(p->eps, n, eps, dev) || !fetch(p->rm, n, rm, dev) || !fetch(p->type, n, type, dev) ||
        !fetch(p->omega, (size_t)T * T, om, dev) || !fetch(p->sigma, (size_t)T * T, sg, dev) ||
        !fetch(p->mu, (size_t)T * T, mu, dev) || !fetch(p->pairs, (size_t)2 * np, pr, dev))
        return bail(DOCK_E_INVALID_ARG);
    for (int a = 0; a < n; a++)
        if (!std::isfinite(q[a]) || !(R[a] > 0.0) || !std::isfinite(R[a]) || !std::isfinite(V[a]) ||
            !(eps[a] >= 0.0) || !std::isfinite(eps[a]) || !std::isfinite(rm[a]) || type[a] < 0 || type[a] >= T)
            return bail(DOCK_E_INVALID_ARG);
    for (size_t t = 0; t < (size_t)T * T; t++)
        if (!std::isfinite(om[t]) || !(sg[t] > 0.0) || !std::isfinite(sg[t]) || !(mu[t] > 0.0) || !std::isfinite(mu[t]))
            return bail(DOCK_E_INVALID_ARG);
    // forward segments (pairs sorted by (i, j), i < j, unique) and reverse segments (by second atom)
    std::vector<int> fwd(n + 1, 0), revc(n + 1, 0), rev(np);
    for (int k = 0; k < np; k++) {
        const int i = pr[2 * k], j = pr[2 * k + 1];
        if (i < 0 || j >= n || i >= j) return bail(DOCK_E_INVALID_ARG);
        if (k > 0 && (pr[2 * k - 2] > i || (pr[2 * k - 2] == i && pr[2 * k - 1] >= j))) return bail(DOCK_E_INVALID_ARG);
        fwd[i + 1]++;
        revc[j + 1]++;
    }
    for (int a = 0; a < n; a++) {
        fwd[a + 1] += fwd[a];
        revc[a + 1] += revc[a];
    }
    {
        std::vector<int> fill(revc.begin(), revc.end() - 1);
        for (int k = 0; k < np; k++) rev[fill[pr[2 * k + 1]]++] = k;   // pair order within each segment
    }
    // one device blob for every array (doubles first, then ints)
    const size_t nd = (size_t)5 * n + (size_t)3 * T * T;
    const size_t ni = (size_t)n + (size_t)2 * np + (size_t)(n + 1) * 2 + (size_t)np;
    if (cudaMalloc(&ctx->blob, sizeof(double) * nd + sizeof(int) * ni + 64) != cudaSuccess) {
        cudaGetLastError();
        return bail(DOCK_E_OOM);
    }
    std::vector<char> host(sizeof(double) * nd + sizeof(int) * ni);
    double* hd = reinterpret_cast<double*>(host.data());
    size_t o = 0;
    auto putd = [&](const std::vector<double>& v) {
        memcpy(hd + o, v.data(), sizeof(double) * v.size());
        o += v.size();
    };
    putd(q);
    putd(R);
    putd(V);
    putd(eps);
    putd(rm);
    putd(om);
    putd(sg);
    putd(mu);
    int* hi = reinterpret_cast<int*>(hd + o);
    size_t oi = 0;
    auto puti = [&](const int* v, size_t cnt) {
        memcpy(hi + oi, v, sizeof(int) * cnt);
        oi += cnt;
    };
    puti(pr.data(), pr.size());   // int2 pairs first (8-byte aligned: nd doubles precede)
    puti(type.data(), n);
    puti(fwd.data(), n + 1);
    puti(revc.data(), n + 1);
    puti(rev.data(), np);
    if (cudaMemcpy(ctx->blob, host.data(), host.size(), cudaMemcpyHostToDevice) != cudaSuccess) return bail(DOCK_E_CUDA);
    const double* bd = static_cast<const double*>(ctx->blob);
    const int* bi = reinterpret_cast<const int*>(bd + nd);
    em::Sys& S = ctx->S;
    S.n = n;
    S.np = np;
    S.T = T;
    S.eps_s = d->eps_s;
    S.rc = d->rc;
    S.tau = 1.0 - 1.0 / d->eps_s;
    S.q = bd;
    S.R = bd + n;
    S.V = bd + 2 * n;
    S.eps = bd + 3 * n;
    S.rm = bd + 4 * n;
    S.omega = bd + 5 * n;
    S.sigma = S.omega + (size_t)T * T;
    S.mu = S.sigma + (size_t)T * T;
    S.pairs = reinterpret_cast<const int2*>(bi);
    S.type = bi + 2 * np;
    S.fwd_off = S.type + n;
    S.rev_off = S.fwd_off + n + 1;
    S.rev_pair = S.rev_off + n + 1;
    *out = ctx;
    return DOCK_OK;
}

dock_status dock_em_eval(dock_em_ctx* ctx, const double* xyz, int n_conf, double* energies, double* forces)
{
    if (!ctx) return DOCK_E_INVALID_ARG;
    if (ctx->dead) return em_fail(ctx, DOCK_E_CUDA, "context unusable after an earlier CUDA error");
    if (!xyz || !energies || n_conf < 0) return em_fail(ctx, DOCK_E_INVALID_ARG, "null input/output or n_conf < 0");
    if (n_conf == 0) return DOCK_OK;
    if (cudaSetDevice(ctx->device) != cudaSuccess) return em_fail(ctx, DOCK_E_CUDA, "cudaSetDevice");
    const em::Sys& S = ctx->S;
    const size_t n = S.n, np = S.np;
    if ((double)n_conf * std::max<size_t>(np, n) > 2e9) return em_fail(ctx, DOCK_E_UNSUPPORTED, "batch too large");
    const int kx = em_ptr_kind(xyz, ctx->device), ke = em_ptr_kind(energies, ctx->device),
              kf = em_ptr_kind(forces, ctx->device);
    if (kx < 0 || ke < 0 || kf < 0) return em_fail(ctx, DOCK_E_INVALID_ARG, "device memory of another device");
    if (kx == 0)
        for (size_t i = 0; i < (size_t)n_conf * n * 3; i++)
            if (!std::isfinite(xyz[i])) return em_fail(ctx, DOCK_E_INVALID_ARG, "non-finite coordinates");
    if (n_conf > ctx->cap_conf) {
        cudaStreamSynchronize(ctx->stream);
        void* keep = ctx->blob;
        ctx->blob = nullptr;
        em_free(ctx);
        ctx->blob = keep;
        ctx->cap_conf = 0;
        const size_t cn = (size_t)n_conf * n, cp = (size_t)n_conf * std::max<size_t>(np, 1);
        ECU(cudaMalloc(&ctx->s, sizeof(double) * cn));
        ECU(cudaMalloc(&ctx->alpha, sizeof(double) * cn));
        ECU(cudaMalloc(&ctx->eself, sizeof(double) * cn));
        ECU(cudaMalloc(&ctx->cfac, sizeof(double) * cn));
        ECU(cudaMalloc(&ctx->dEdr, sizeof(double) * cp));
        ECU(cudaMalloc(&ctx->e_pair, sizeof(double2) * cp));
        ECU(cudaMalloc(&ctx->dal, sizeof(double2) * cp));
        ECU(cudaMalloc(&ctx->dsd, sizeof(double2) * cp));
        ECU(cudaMalloc(&ctx->d_x, sizeof(double) * cn * 3));
        ECU(cudaMalloc(&ctx->d_e, sizeof(double) * 3 * n_conf));
        ECU(cudaMalloc(&ctx->d_f, sizeof(double) * cn * 3));
        ctx->cap_conf = n_conf;
    }
    cudaStream_t st = ctx->stream;
    const double* dx = xyz;
    if (kx == 0) {
        ECU(cudaMemcpyAsync(ctx->d_x, xyz, sizeof(double) * n_conf * n * 3, cudaMemcpyHostToDevice, st));
        dx = ctx->d_x;
    }
    double* de = ke == 1 ? energies : ctx->d_e;
    double* df = forces ? (kf == 1 ? forces : ctx->d_f) : nullptr;
    const long long na = (long long)n_conf * n, npc = (long long)n_conf * np;
    const int B = 128;
    ECU(cudaEventRecord(ctx->ev[0], st));
    const long long naw = na * 32;   // warp per (conformation, atom)
    em::k_em_self<<<(unsigned)((naw + B - 1) / B), B, 0, st>>>(S, dx, n_conf, ctx->s, ctx->alpha, ctx->eself,
                                                                ctx->dsd);
    if (np > 0)
        em::k_em_pair<<<(unsigned)((npc + B - 1) / B), B, 0, st>>>(S, dx, n_conf, ctx->alpha, ctx->e_pair, ctx->dEdr,
                                                                 ctx->dal);
    if (df) {
        em::k_em_chain<<<(unsigned)((naw + B - 1) / B), B, 0, st>>>(S, n_conf, ctx->s, ctx->dal, ctx->cfac);
        em::k_em_force<<<(unsigned)((naw + B - 1) / B), B, 0, st>>>(S, dx, n_conf, ctx->dEdr, ctx->dsd, ctx->cfac,
                                                                     df);
    }
    em::k_em_energy<<<n_conf, 256, 0, st>>>(S.n, S.np, ctx->eself, ctx->e_pair, de);
    ECU(cudaGetLastError());
    ECU(cudaEventRecord(ctx->ev[1], st));
    ctx->ev_valid = true;
    if (ke == 0) ECU(cudaMemcpyAsync(energies, de, sizeof(double) * 3 * n_conf, cudaMemcpyDeviceToHost, st));
    if (forces && kf == 0) ECU(cudaMemcpyAsync(forces, df, sizeof(double) * n_conf * n * 3, cudaMemcpyDeviceToHost, st));
    ECU(cudaStreamSynchronize(st));
    return DOCK_OK;
}

}  // extern "C"

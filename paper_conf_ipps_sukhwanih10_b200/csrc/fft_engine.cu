// FFT correlation engine (see dock_fft.h).
#include <cufft.h>

#include <algorithm>
#include <cstddef>

#define DOCK_LAUNCHER_TU
#include "dock_fft.h"
#include "dock_kernels.cuh"   // dk::RB (k_voxelize weight layout)

namespace {

// receptor channel p, unpadded: R[p][z][y][x] = rec[p][z][y][x] (the padded copy starts at the origin)
__global__ void k_fft_unpad(const float* __restrict__ rec, float* __restrict__ R, int Xp, int Yp, int Zp, int nx,
                            int ny, int nz, int P)
{
    const size_t total = static_cast<size_t>(P) * nz * ny * nx;
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<size_t>(gridDim.x) * blockDim.x) {
        const int x = static_cast<int>(i % nx);
        size_t r = i / nx;
        const int y = static_cast<int>(r % ny);
        r /= ny;
        const int z = static_cast<int>(r % nz);
        const int p = static_cast<int>(r / nz);
        R[i] = rec[((static_cast<size_t>(p) * Zp + z) * Yp + y) * Xp + x];
    }
}

// ligand grids zero-padded to the receptor grid: Lpad[b][p][vz][vy][vx] = Lw(slot0 + b, p, v); the rest of
// Lpad is zeroed by the caller
__global__ void k_fft_scatter(const float* __restrict__ Lw, float* __restrict__ Lpad, int slot0, int n, int P, int m,
                              int nx, int ny, int nz)
{
    const int m3 = m * m * m;
    const int total = n * P * m3;
    for (int i = blockIdx.x * blockDim.x + threadIdx.x; i < total; i += gridDim.x * blockDim.x) {
        const int v = i % m3, p = (i / m3) % P, b = i / (m3 * P);
        const int s = slot0 + b;
        const int vx = v % m, vy = (v / m) % m, vz = v / (m * m);
        const float w = Lw[((static_cast<size_t>(s / dk::RB) * P + p) * m3 + v) * dk::RB + s % dk::RB];
        Lpad[((static_cast<size_t>(b) * P + p) * nz + vz) * ny * static_cast<size_t>(nx) + static_cast<size_t>(vy) * nx +
             vx] = w;
    }
}

// Shat[b][i] = scale * sum_p Rhat[p][i] * conj(Lhat[b][p][i])   (cross-correlation theorem)
__global__ void k_fft_mac(const float2* __restrict__ Rhat, const float2* __restrict__ Lhat, float2* __restrict__ Shat,
                          size_t nc, int n, int P, float scale)
{
    const size_t total = static_cast<size_t>(n) * nc;
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<size_t>(gridDim.x) * blockDim.x) {
        const size_t c = i % nc, b = i / nc;
        float re = 0.f, im = 0.f;
        for (int p = 0; p < P; p++) {
            const float2 r = Rhat[static_cast<size_t>(p) * nc + c];
            const float2 l = Lhat[(b * P + p) * nc + c];
            re += r.x * l.x + r.y * l.y;   // r * conj(l)
            im += r.y * l.x - r.x * l.y;
        }
        Shat[i] = make_float2(re * scale, im * scale);
    }
}

}  // namespace

struct DockFft {
    const float* rec_key = nullptr;   // receptor the cached transform belongs to
    int nx = 0, ny = 0, nz = 0, P = 0;
    float2* Rhat = nullptr;           // [P][nz][ny][nx/2+1]
    float* Lpad = nullptr;            // [B][P][nz][ny][nx]
    float2* Lhat = nullptr;           // [B][P][nc]
    float2* Shat = nullptr;           // [B][nc]
    int cap = 0;                      // B the buffers hold
    int m_last = 0;                   // ligand size of the last scatter (Lpad outside [0,m)^3 stays zero)
    struct Plans {
        cufftHandle fwd = 0, inv = 0;   // batched R2C (n*P) and C2R (n) plans
        int n = 0;
    } plans[2];                         // the full chunk and the tail chunk of a call
};

DockFft* dock_fft_create() { return new DockFft(); }

static void free_bufs(DockFft* f)
{
    cudaFree(f->Lpad);
    cudaFree(f->Lhat);
    cudaFree(f->Shat);
    f->Lpad = nullptr;
    f->Lhat = nullptr;
    f->Shat = nullptr;
    f->cap = 0;
    f->m_last = 0;
    for (auto& pl : f->plans) {
        if (pl.n) {
            cufftDestroy(pl.fwd);
            cufftDestroy(pl.inv);
            pl.n = 0;
        }
    }
}

void dock_fft_destroy(DockFft* f)
{
    if (!f) return;
    free_bufs(f);
    cudaFree(f->Rhat);
    delete f;
}

int dock_fft_batch(int nx, int ny, int nz, int P)
{
    const double cells = double(nx) * ny * nz;
    const double per = cells * 4.0 * P + cells * 4.2 * P + cells * 4.2;   // Lpad + Lhat + Shat per grid
    return (int)std::max(1.0, std::min(64.0, 6.0e9 / per));
}

#define CK(x)                                         \
    do {                                              \
        cudaError_t e_ = (x);                         \
        if (e_ != cudaSuccess) return e_;             \
    } while (0)
#define FK(x)                                         \
    do {                                              \
        if ((x) != CUFFT_SUCCESS) return cudaErrorUnknown; \
    } while (0)

cudaError_t dock_fft_grids(DockFft* f, const float* rec, int Xp, int Yp, int Zp, int nx, int ny, int nz, int P, int m,
                           const float* Lw, int slot0, int n, float* S, cudaStream_t st)
{
    const size_t cells = static_cast<size_t>(nx) * ny * nz;
    const size_t nc = static_cast<size_t>(nz) * ny * (nx / 2 + 1);
    int dims[3] = {nz, ny, nx};
    if (f->rec_key != rec || f->nx != nx || f->ny != ny || f->nz != nz || f->P != P) {
        // receptor transform, once per receptor
        free_bufs(f);
        cudaFree(f->Rhat);
        f->Rhat = nullptr;
        float* R = nullptr;
        CK(cudaMalloc(&R, sizeof(float) * cells * P));
        CK(cudaMalloc(&f->Rhat, sizeof(float2) * nc * P));
        k_fft_unpad<<<1024, 256, 0, st>>>(rec, R, Xp, Yp, Zp, nx, ny, nz, P);
        CK(cudaGetLastError());
        cufftHandle h;
        FK(cufftPlanMany(&h, 3, dims, nullptr, 1, 0, nullptr, 1, 0, CUFFT_R2C, P));
        FK(cufftSetStream(h, st));
        const cufftResult r = cufftExecR2C(h, R, reinterpret_cast<cufftComplex*>(f->Rhat));
        CK(cudaStreamSynchronize(st));
        cufftDestroy(h);
        cudaFree(R);
        if (r != CUFFT_SUCCESS) return cudaErrorUnknown;
        f->rec_key = rec;
        f->nx = nx;
        f->ny = ny;
        f->nz = nz;
        f->P = P;
    }
    if (n > f->cap) {
        free_bufs(f);
        CK(cudaMalloc(&f->Lpad, sizeof(float) * cells * P * n));
        CK(cudaMalloc(&f->Lhat, sizeof(float2) * nc * P * n));
        CK(cudaMalloc(&f->Shat, sizeof(float2) * nc * n));
        f->cap = n;
    }
    // plans for this batch size: two cached (the full chunk and the tail of a call)
    DockFft::Plans* pl = nullptr;
    for (auto& c : f->plans)
        if (c.n == n) pl = &c;
    if (!pl) {
        pl = f->plans[0].n == 0 ? &f->plans[0] : &f->plans[1];
        if (pl->n) {
            cufftDestroy(pl->fwd);
            cufftDestroy(pl->inv);
            pl->n = 0;
        }
        FK(cufftPlanMany(&pl->fwd, 3, dims, nullptr, 1, 0, nullptr, 1, 0, CUFFT_R2C, P * n));
        FK(cufftPlanMany(&pl->inv, 3, dims, nullptr, 1, 0, nullptr, 1, 0, CUFFT_C2R, n));
        pl->n = n;
    }
    FK(cufftSetStream(pl->fwd, st));
    FK(cufftSetStream(pl->inv, st));
    // the scatter only writes [0,m)^3 of every padded grid: zero the buffer only when m changes
    if (m != f->m_last) {
        CK(cudaMemsetAsync(f->Lpad, 0, sizeof(float) * cells * P * f->cap, st));
        f->m_last = m;
    }
    const int m3 = m * m * m;
    k_fft_scatter<<<std::max(1, std::min(1024, (n * P * m3 + 255) / 256)), 256, 0, st>>>(Lw, f->Lpad, slot0, n, P, m,
                                                                                      nx, ny, nz);
    CK(cudaGetLastError());
    FK(cufftExecR2C(pl->fwd, f->Lpad, reinterpret_cast<cufftComplex*>(f->Lhat)));
    k_fft_mac<<<2048, 256, 0, st>>>(f->Rhat, f->Lhat, f->Shat, nc, n, P, 1.0f / static_cast<float>(cells));
    CK(cudaGetLastError());
    FK(cufftExecC2R(pl->inv, reinterpret_cast<cufftComplex*>(f->Shat), S));
    return cudaGetLastError();
}

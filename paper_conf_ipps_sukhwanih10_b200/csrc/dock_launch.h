// dock_launch.h -- launchers of the correlation kernels.  Each family is instantiated in its own
// translation unit (launch_*.cu, compiled in parallel); dock.cu holds the host logic and the small
// kernels.  Internal to libdock.so (not part of the C ABI).
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include "dock_kernels.cuh"
#include "dock_tc.cuh"
#include "dock_sparse.cuh"

// FP32 FFMA engine k_corr<m, grid>
cudaError_t dock_launch_ffma(int m, bool grid, const CUtensorMap& tmap, int smem, const dk::CorrArgs& a, int nblocks,
                             cudaStream_t st);
// tcgen05 variant 1 k_corr_tc<m, grid> (one channel group, resident boxes, NTT = 128, Q = 4)
cudaError_t dock_launch_tc1(int m, bool grid, const CUtensorMap& tmap, const CUtensorMap& tmap_pair,
                            const CUtensorMap& tmap_b, int smem, const tc::TcArgs& a, int nblocks, cudaStream_t st);
// tcgen05 variant 2 k_corr_tcs<m, ntt, q(ntt), grid> (streamed planes); ntt in {64, 128, 160}
cudaError_t dock_launch_tcs64(int m, bool grid, const CUtensorMap& tmap, const CUtensorMap& tmap_pair, int smem,
                              const tc::TcArgs& a, int nblocks, cudaStream_t st);
cudaError_t dock_launch_tcs128(int m, bool grid, const CUtensorMap& tmap, const CUtensorMap& tmap_pair, int smem,
                               const tc::TcArgs& a, int nblocks, cudaStream_t st);
cudaError_t dock_launch_tcs160(int m, bool grid, const CUtensorMap& tmap, const CUtensorMap& tmap_pair, int smem,
                               const tc::TcArgs& a, int nblocks, cudaStream_t st);

// sparse-ligand engine k_corr_sparse<xts, zt, grid> (dock_sparse.cuh); xts = translations per lane along x
cudaError_t dock_launch_sparse2(int zt, bool grid, const CUtensorMap& gmap, int smem, const sp::SpArgs& a, int nblocks,
                                cudaStream_t st);
cudaError_t dock_launch_sparse4(int zt, bool grid, const CUtensorMap& gmap, int smem, const sp::SpArgs& a, int nblocks,
                                cudaStream_t st);
cudaError_t dock_launch_sparse5(int zt, bool grid, const CUtensorMap& gmap, int smem, const sp::SpArgs& a, int nblocks,
                                cudaStream_t st);
inline cudaError_t dock_launch_sparse(int xts, int zt, bool grid, const CUtensorMap& gmap, int smem,
                                      const sp::SpArgs& a, int nblocks, cudaStream_t st)
{
    switch (xts) {
        case 2: return dock_launch_sparse2(zt, grid, gmap, smem, a, nblocks, st);
        case 4: return dock_launch_sparse4(zt, grid, gmap, smem, a, nblocks, st);
        case 5: return dock_launch_sparse5(zt, grid, gmap, smem, a, nblocks, st);
        default: return cudaErrorInvalidValue;
    }
}

// rows per tile of the streamed kernel for a row width: Q * NTT <= 512 TMEM columns
constexpr int tcs_q(int ntt) { return ntt == 64 ? 8 : ntt == 160 ? 3 : 4; }

inline cudaError_t dock_launch_tcs(int m, int ntt, bool grid, const CUtensorMap& tmap, const CUtensorMap& tmap_pair,
                                   int smem, const tc::TcArgs& a, int nblocks, cudaStream_t st)
{
    switch (ntt) {
        case 64: return dock_launch_tcs64(m, grid, tmap, tmap_pair, smem, a, nblocks, st);
        case 128: return dock_launch_tcs128(m, grid, tmap, tmap_pair, smem, a, nblocks, st);
        case 160: return dock_launch_tcs160(m, grid, tmap, tmap_pair, smem, a, nblocks, st);
        default: return cudaErrorInvalidValue;
    }
}

// m -> template dispatch shared by the launcher TUs
#define DOCK_DISPATCH_M(m, CALL)                 \
    switch (m) {                                 \
        case 1: return CALL(1);                  \
        case 2: return CALL(2);                  \
        case 3: return CALL(3);                  \
        case 4: return CALL(4);                  \
        case 5: return CALL(5);                  \
        case 6: return CALL(6);                  \
        case 7: return CALL(7);                  \
        case 8: return CALL(8);                  \
        default: return cudaErrorInvalidValue;   \
    }

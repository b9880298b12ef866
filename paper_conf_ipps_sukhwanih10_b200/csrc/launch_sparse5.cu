// sparse-ligand engine instantiations (k_corr_sparse, dock_sparse.cuh) for 5 translations per lane along x
// (planes per warp ZT = 1).
#define DOCK_LAUNCHER_TU
#include "dock_launch.h"

template <int ZT, bool GRID>
static cudaError_t launch_t(const CUtensorMap& gmap, int smem, const sp::SpArgs& a, int nblocks, cudaStream_t st)
{
    auto kern = sp::k_corr_sparse<5, ZT, GRID>;
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    if (e != cudaSuccess) return e;
    kern<<<nblocks, sp::NTHREADS, smem, st>>>(gmap, a);
    return cudaGetLastError();
}

cudaError_t dock_launch_sparse5(int zt, bool grid, const CUtensorMap& gmap, int smem, const sp::SpArgs& a,
                                int nblocks, cudaStream_t st)
{
    if (zt != 1) return cudaErrorInvalidValue;
    return grid ? launch_t<1, true>(gmap, smem, a, nblocks, st) : launch_t<1, false>(gmap, smem, a, nblocks, st);
}

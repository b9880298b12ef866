// FP32 FFMA correlation kernel instantiations (see dock_kernels.cuh).
#define DOCK_LAUNCHER_TU
#include "dock_launch.h"

template <int M, bool GRID>
static cudaError_t launch_t(const CUtensorMap& tmap, int smem, const dk::CorrArgs& a, int nblocks, cudaStream_t st)
{
    auto kern = dk::k_corr<M, GRID>;
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    if (e != cudaSuccess) return e;
    kern<<<nblocks, dk::NTHREADS, smem, st>>>(tmap, a);
    return cudaGetLastError();
}

cudaError_t dock_launch_ffma(int m, bool grid, const CUtensorMap& tmap, int smem, const dk::CorrArgs& a, int nblocks,
                             cudaStream_t st)
{
#define CALL_G(M) launch_t<M, true>(tmap, smem, a, nblocks, st)
#define CALL_S(M) launch_t<M, false>(tmap, smem, a, nblocks, st)
    if (grid) { DOCK_DISPATCH_M(m, CALL_G) }
    DOCK_DISPATCH_M(m, CALL_S)
}

// tcgen05 variant 1 instantiations (k_corr_tc, dock_tc.cuh).
#define DOCK_LAUNCHER_TU
#include "dock_launch.h"

template <int M, bool GRID>
static cudaError_t launch_t(const CUtensorMap& tmap, const CUtensorMap& tmap_pair, const CUtensorMap& tmap_b,
                            int smem, const tc::TcArgs& a, int nblocks, cudaStream_t st)
{
    auto kern = tc::k_corr_tc<M, GRID>;
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    if (e != cudaSuccess) return e;
    kern<<<nblocks, (3 + a.nepi) * 32, smem, st>>>(tmap, tmap_pair, tmap_b, a);   // + receptor producer warp
    return cudaGetLastError();
}

cudaError_t dock_launch_tc1(int m, bool grid, const CUtensorMap& tmap, const CUtensorMap& tmap_pair,
                            const CUtensorMap& tmap_b, int smem, const tc::TcArgs& a, int nblocks, cudaStream_t st)
{
#define CALL_G(M) launch_t<M, true>(tmap, tmap_pair, tmap_b, smem, a, nblocks, st)
#define CALL_S(M) launch_t<M, false>(tmap, tmap_pair, tmap_b, smem, a, nblocks, st)
    if (grid) { DOCK_DISPATCH_M(m, CALL_G) }
    DOCK_DISPATCH_M(m, CALL_S)
}

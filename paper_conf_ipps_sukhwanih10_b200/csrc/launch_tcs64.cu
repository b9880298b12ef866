// tcgen05 variant 2 instantiations (k_corr_tcs, dock_tc.cuh) for 64 translations per MMA row.
#define DOCK_LAUNCHER_TU
#include "dock_launch.h"

template <int M, bool GRID>
static cudaError_t launch_t(const CUtensorMap& tmap, const CUtensorMap& tmap_pair, int smem, const tc::TcArgs& a,
                            int nblocks, cudaStream_t st)
{
    auto kern = tc::k_corr_tcs<M, 64, tcs_q(64), GRID>;
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    if (e != cudaSuccess) return e;
    kern<<<nblocks, (3 + a.nepi) * 32, smem, st>>>(tmap, tmap_pair, a);   // + receptor producer warp
    return cudaGetLastError();
}

cudaError_t dock_launch_tcs64(int m, bool grid, const CUtensorMap& tmap, const CUtensorMap& tmap_pair, int smem,
                              const tc::TcArgs& a, int nblocks, cudaStream_t st)
{
#define CALL_G(M) launch_t<M, true>(tmap, tmap_pair, smem, a, nblocks, st)
#define CALL_S(M) launch_t<M, false>(tmap, tmap_pair, smem, a, nblocks, st)
    if (grid) { DOCK_DISPATCH_M(m, CALL_G) }
    DOCK_DISPATCH_M(m, CALL_S)
}

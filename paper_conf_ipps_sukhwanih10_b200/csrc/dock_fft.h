// dock_fft.h -- FFT correlation engine (the paper's FFT method P:L156-163, kept as the
// comparison point of the direct-vs-FFT crossover P:L485-502).  Internal to libdock.so.
//
// S[t] = sum_p IFFT( FFT(R_p) * conj(FFT(Lw_p zero-padded to the receptor grid)) )[t] / (nx ny nz), the
// cyclic cross-correlation of reading Q1/Q2.  cuFFT does the transforms (a plain library FFT, like
// cuBLAS for a plain GEMM); the ligand scatter and the frequency-domain multiply-accumulate over the
// channels are this library's kernels.  FP32 throughout: FFT rounding is global (relative to the grid
// norm), not per cell like direct correlation, so its score-grid tolerance is stated against max A.
#pragma once
#include <cuda_runtime.h>

struct DockFft;

DockFft* dock_fft_create();
void dock_fft_destroy(DockFft* f);
// Score grids S[n][nz][ny][nx] of slots [slot0, slot0 + n) from the folded weights Lw
// ([ceil(.)/RB][P][m^3][RB], k_voxelize layout); rec = the cyclic-halo padded receptor [P][Zp][Yp][Xp].
// Returns the first CUDA / cuFFT failure as cudaErrorUnknown (cuFFT) or the CUDA error.
cudaError_t dock_fft_grids(DockFft* f, const float* rec, int Xp, int Yp, int Zp, int nx, int ny, int nz, int P, int m,
                           const float* Lw, int slot0, int n, float* S, cudaStream_t st);
// largest batch of grids one dock_fft_grids call should take for this problem size (memory bound)
int dock_fft_batch(int nx, int ny, int nz, int P);

// fma_bench.cu -- FP32 FMA issue-rate microbenchmark on sm_100a (design evidence for k_corr).
// Variants: 3-register FFMA (acc += w*r with w reused), FFMA with a constant-bank operand,
// FFMA2 (fma.rn.f32x2).  Prints TFLOP/s per variant at the observed clock.
#include <cstdio>
#include <cuda_runtime.h>

constexpr int NACC = 32;
constexpr int ITERS = 4096;

__constant__ float cw[64];

// acc[i] += w[j] * r[i]: the k_corr pattern (w reused across 8 accumulators).
__global__ void __launch_bounds__(256) k_reg(float* out, float seed)
{
    float r[8], w[4], acc[NACC];
#pragma unroll
    for (int i = 0; i < 8; i++) r[i] = seed * (threadIdx.x + i);
#pragma unroll
    for (int i = 0; i < 4; i++) w[i] = seed * (i + 1);
#pragma unroll
    for (int i = 0; i < NACC; i++) acc[i] = 0.f;
    for (int it = 0; it < ITERS; it++) {
#pragma unroll
        for (int j = 0; j < 4; j++)
#pragma unroll
            for (int i = 0; i < 8; i++) acc[j * 8 + i] = fmaf(w[j], r[i], acc[j * 8 + i]);
#pragma unroll
        for (int i = 0; i < 8; i++) r[i] = __int_as_float(__float_as_int(r[i]) ^ 1);
    }
    float s = 0;
#pragma unroll
    for (int i = 0; i < NACC; i++) s += acc[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

__global__ void __launch_bounds__(256) k_const(float* out, float seed)
{
    float r[8], acc[NACC];
#pragma unroll
    for (int i = 0; i < 8; i++) r[i] = seed * (threadIdx.x + i);
#pragma unroll
    for (int i = 0; i < NACC; i++) acc[i] = 0.f;
    for (int it = 0; it < ITERS; it++) {
#pragma unroll
        for (int j = 0; j < 4; j++)
#pragma unroll
            for (int i = 0; i < 8; i++) acc[j * 8 + i] = fmaf(cw[j], r[i], acc[j * 8 + i]);
#pragma unroll
        for (int i = 0; i < 8; i++) r[i] = __int_as_float(__float_as_int(r[i]) ^ 1);
    }
    float s = 0;
#pragma unroll
    for (int i = 0; i < NACC; i++) s += acc[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

__device__ __forceinline__ unsigned long long f2(float2 v) { return *reinterpret_cast<unsigned long long*>(&v); }

__global__ void __launch_bounds__(256) k_f2(float* out, float seed)
{
    float2 r[4], w[4];
    unsigned long long acc[NACC / 2];
#pragma unroll
    for (int i = 0; i < 4; i++) r[i] = make_float2(seed * (threadIdx.x + 2 * i), seed * (threadIdx.x + 2 * i + 1));
#pragma unroll
    for (int i = 0; i < 4; i++) w[i] = make_float2(seed * (i + 1), seed * (i + 1));
#pragma unroll
    for (int i = 0; i < NACC / 2; i++) acc[i] = 0ull;
    for (int it = 0; it < ITERS; it++) {
#pragma unroll
        for (int j = 0; j < 4; j++)
#pragma unroll
            for (int i = 0; i < 4; i++)
                asm volatile("fma.rn.f32x2 %0, %1, %2, %0;" : "+l"(acc[j * 4 + i]) : "l"(f2(w[j])), "l"(f2(r[i])));
#pragma unroll
        for (int i = 0; i < 4; i++) r[i].x = __int_as_float(__float_as_int(r[i].x) ^ 1);
    }
    float s = 0;
#pragma unroll
    for (int i = 0; i < NACC / 2; i++) {
        float2 v = *reinterpret_cast<float2*>(&acc[i]);
        s += v.x + v.y;
    }
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

template <typename K>
double run(K kern, float* out, int blocks, int threads, const char* name)
{
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    kern<<<blocks, threads>>>(out, 1e-7f);
    cudaEventRecord(a);
    const int reps = 5;
    for (int i = 0; i < reps; i++) kern<<<blocks, threads>>>(out, 1e-7f);
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    float ms;
    cudaEventElapsedTime(&ms, a, b);
    double flops = 2.0 * NACC * ITERS * (double)blocks * threads * reps;
    double tf = flops / (ms * 1e-3) / 1e12;
    int clk = 0;
    cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    printf("%-10s blocks=%d threads=%d  %.2f TFLOP/s  (%.3f ms/launch)\n", name, blocks, threads, tf, ms / reps);
    return tf;
}

int main()
{
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    float h[64];
    for (int i = 0; i < 64; i++) h[i] = 1e-7f * (i + 1);
    cudaMemcpyToSymbol(cw, h, sizeof(h));
    float* out;
    cudaMalloc(&out, sizeof(float) * sms * 8 * 256);
    for (int occ : {2, 4, 8}) {
        run(k_reg, out, sms * occ, 256, "ffma_reg");
        run(k_const, out, sms * occ, 256, "ffma_const");
        run(k_f2, out, sms * occ, 256, "ffma2");
    }
    printf("peak at 1965 MHz: %.2f TFLOP/s\n", sms * 128 * 2 * 1.965e9 / 1e12);
    return 0;
}

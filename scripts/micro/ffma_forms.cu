// FFMA operand-form throughput on sm_100a: 3-register, register + immediate,
// register + uniform register (coefficient from LDCU), register + shared-memory
// broadcast.  8 independent accumulator chains per thread; 16 warps/SM.
#include <cstdio>
#include <cuda_runtime.h>
#define N_IT 4096
__constant__ float CC[64];
extern "C" __global__ void f_reg3(float* out, float a0, float b0) {
    float x[8], c[8], acc[8];
    for (int i = 0; i < 8; i++) { x[i] = a0 + i + threadIdx.x; c[i] = b0 * (i + 1); acc[i] = 0; }
    #pragma unroll 1
    for (int it = 0; it < N_IT; it++) {
        #pragma unroll
        for (int r = 0; r < 8; r++)
            #pragma unroll
            for (int i = 0; i < 8; i++) acc[i] = fmaf(x[(i + r) & 7], c[(i * 3 + r) & 7], acc[i]);
    }
    float s = 0; for (int i = 0; i < 8; i++) s += acc[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}
extern "C" __global__ void f_imm(float* out, float a0, float b0) {
    float x[8], acc[8];
    for (int i = 0; i < 8; i++) { x[i] = a0 + i + threadIdx.x; acc[i] = 0; }
    #pragma unroll 1
    for (int it = 0; it < N_IT; it++) {
        #pragma unroll
        for (int r = 0; r < 8; r++)
            #pragma unroll
            for (int i = 0; i < 8; i++) acc[i] = fmaf(x[(i + r) & 7], 1.0f + 0.125f * ((i * 3 + r) & 7), acc[i]);
    }
    float s = 0; for (int i = 0; i < 8; i++) s += acc[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}
extern "C" __global__ void f_ucst(float* out, float a0, float b0) {
    float x[8], acc[8];
    for (int i = 0; i < 8; i++) { x[i] = a0 + i + threadIdx.x; acc[i] = 0; }
    #pragma unroll 1
    for (int it = 0; it < N_IT; it++) {
        const int base = (it & 3) * 16;
        #pragma unroll
        for (int r = 0; r < 8; r++)
            #pragma unroll
            for (int i = 0; i < 8; i++) acc[i] = fmaf(x[(i + r) & 7], CC[base + ((i * 3 + r) & 15)], acc[i]);
    }
    float s = 0; for (int i = 0; i < 8; i++) s += acc[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}
__constant__ float2 CC2[64];
extern "C" __global__ void f_ffma2_reg(float* out, float a0, float b0) {
    float2 x[8], c[8], acc[8];
    for (int i = 0; i < 8; i++) { x[i] = make_float2(a0 + i + threadIdx.x, a0 - i); c[i] = make_float2(b0 * (i + 1), b0 - i); acc[i] = make_float2(0.f, 0.f); }
    #pragma unroll 1
    for (int it = 0; it < N_IT / 2; it++) {
        #pragma unroll
        for (int r = 0; r < 8; r++)
            #pragma unroll
            for (int i = 0; i < 8; i++) acc[i] = __ffma2_rn(x[(i + r) & 7], c[(i * 3 + r) & 7], acc[i]);
    }
    float s = 0; for (int i = 0; i < 8; i++) s += acc[i].x + acc[i].y;
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}
extern "C" __global__ void f_ffma2_cst(float* out, float a0, float b0) {
    float2 x[8], acc[8];
    for (int i = 0; i < 8; i++) { x[i] = make_float2(a0 + i + threadIdx.x, a0 - i); acc[i] = make_float2(0.f, 0.f); }
    #pragma unroll 1
    for (int it = 0; it < N_IT / 2; it++) {
        #pragma unroll
        for (int r = 0; r < 8; r++)
            #pragma unroll
            for (int i = 0; i < 8; i++) acc[i] = __ffma2_rn(x[(i + r) & 7], CC2[(i * 3 + r) & 63], acc[i]);
    }
    float s = 0; for (int i = 0; i < 8; i++) s += acc[i].x + acc[i].y;
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}
int main() {
    float* d; cudaMalloc(&d, 148 * 8 * 256 * 4);
    float h[64]; for (int i = 0; i < 64; i++) h[i] = 1.0f + i * 0.01f;
    cudaMemcpyToSymbol(CC, h, sizeof h);
    cudaMemcpyToSymbol(CC2, h, sizeof h);
    int sm; cudaDeviceGetAttribute(&sm, cudaDevAttrMultiProcessorCount, 0);
    int clk; cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    struct { const char* n; void (*k)(float*, float, float); } ks[] = {{"reg3", f_reg3}, {"imm", f_imm}, {"ucst", f_ucst}, {"ffma2_reg", f_ffma2_reg}, {"ffma2_cst", f_ffma2_cst}};
    for (auto& k : ks) {
        for (int rep = 0; rep < 2; rep++) {
            cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
            cudaEventRecord(a);
            k.k<<<sm * 8, 256>>>(d, 1.0f, 0.5f);
            cudaEventRecord(b); cudaEventSynchronize(b);
            float ms; cudaEventElapsedTime(&ms, a, b);
            double fl = 2.0 * sm * 8 * 256 * (double)N_IT * 64;
            if (rep) printf("%-5s %.2f TFLOP/s (%.1f%% of %d SMs x 128 x 2 x %.0f MHz)\n", k.n, fl / ms / 1e9,
                            100.0 * fl / ms / 1e9 / (sm * 256.0 * clk / 1e6), sm, clk / 1e3);
        }
    }
    return 0;
}

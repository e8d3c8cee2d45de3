// Microbenchmark (development aid): FP64 / integer pipe latency and throughput on this GPU.
// nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/fp64_micro tools/fp64_micro.cu
#include <cstdio>
#include <cuda_runtime.h>

template <int ILP>
__global__ void dfma_chain(double* out, int iters, double a, double b) {
    double x[ILP];
#pragma unroll
    for (int i = 0; i < ILP; ++i) x[i] = threadIdx.x * 1e-3 + i;
    for (int it = 0; it < iters; ++it) {
#pragma unroll
        for (int i = 0; i < ILP; ++i) x[i] = fma(x[i], a, b);
    }
    double s = 0;
#pragma unroll
    for (int i = 0; i < ILP; ++i) s += x[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

template <int ILP>
__global__ void imad_chain(unsigned* out, int iters, unsigned a, unsigned b) {
    unsigned x[ILP];
#pragma unroll
    for (int i = 0; i < ILP; ++i) x[i] = threadIdx.x + i;
    for (int it = 0; it < iters; ++it) {
#pragma unroll
        for (int i = 0; i < ILP; ++i) {
            unsigned long long p = (unsigned long long)x[i] * a;
            x[i] = (unsigned)(p >> 32) ^ (unsigned)p ^ b;
        }
    }
    unsigned s = 0;
#pragma unroll
    for (int i = 0; i < ILP; ++i) s += x[i];
    out[blockIdx.x * blockDim.x + threadIdx.x] = s;
}

__global__ void ddiv_chain(double* out, int iters, double a) {
    double x = threadIdx.x + 1.5;
    for (int it = 0; it < iters; ++it) x = __ddiv_rn(a, x) + 1.0;
    out[blockIdx.x * blockDim.x + threadIdx.x] = x;
}

template <class F>
float timeit(F f) {
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    f();
    cudaEventRecord(e0);
    f();
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    return ms;
}

int main() {
    int sms;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    int clk;
    cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    double* d;
    unsigned* u;
    cudaMalloc(&d, 1 << 26);
    cudaMalloc(&u, 1 << 26);
    const int iters = 4096;
    // latency: one warp per SM, ILP 1
    float ms = timeit([&] { dfma_chain<1><<<sms, 32>>>(d, iters, 1.0000001, 1e-9); });
    printf("DFMA dependent latency ~ %.1f cycles (clock %d kHz)\n", ms * 1e-3 * clk * 1e3 / iters, clk);
    ms = timeit([&] { imad_chain<1><<<sms, 32>>>(u, iters, 0xD2511F53u, 7); });
    printf("IMAD.WIDE+LOP3 round latency ~ %.1f cycles\n", ms * 1e-3 * clk * 1e3 / iters);
    ms = timeit([&] { ddiv_chain<<<sms, 32>>>(d, iters, 3.0); });
    printf("DDIV(+DADD) dependent latency ~ %.1f cycles\n", ms * 1e-3 * clk * 1e3 / iters);
    // throughput: many warps, ILP 4
    for (int warps : {4, 8, 16, 32, 64}) {
        ms = timeit([&] { dfma_chain<4><<<sms, 32 * warps>>>(d, iters, 1.0000001, 1e-9); });
        double ops = (double)sms * 32 * warps * iters * 4;
        printf("DFMA throughput, %2d warps/SM: %.1f DFMA/clk/SM\n", warps, ops / (ms * 1e-3) / (clk * 1e3) / sms);
    }
    for (int warps : {4, 8, 16, 32}) {
        ms = timeit([&] { imad_chain<4><<<sms, 32 * warps>>>(u, iters, 0xD2511F53u, 7); });
        double ops = (double)sms * 32 * warps * iters * 4;
        printf("IMAD.WIDE+LOP3 rounds, %2d warps/SM: %.1f rounds/clk/SM\n", warps, ops / (ms * 1e-3) / (clk * 1e3) / sms);
    }
    return 0;
}

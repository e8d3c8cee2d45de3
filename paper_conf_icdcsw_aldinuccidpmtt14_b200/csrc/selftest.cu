// selftest.cu — AOT (nvcc, sm_100a) kernels exercising the SSA kernel's own device primitives
// (device/cwc_rng.cuh, the very file embedded into every NVRTC-compiled SSA kernel), so the GPU
// tests can compare Philox4x32-10, the 52-bit uniforms and CWC-log bit for bit with the oracle.
// Compiled with -fmad=false like the NVRTC kernels.
#include <cuda_runtime.h>

#include <cstdint>
#include <vector>

#include "cwc.h"
#include "device/cwc_params.h"
#include "device/cwc_rng.cuh"
#include "runtime.hpp"

namespace {

__global__ void k_philox(int64_t n, const uint32_t* ctr, const uint32_t* key, uint32_t* out) {
    int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= n) return;
    cwc_round_keys rk;
    for (int r = 0; r < 10; ++r) {
        rk.k0[r] = key[2 * i] + (uint32_t)r * CWC_PHILOX_W0;
        rk.k1[r] = key[2 * i + 1] + (uint32_t)r * CWC_PHILOX_W1;
    }
    unsigned int c0 = ctr[4 * i], c1 = ctr[4 * i + 1], c2 = ctr[4 * i + 2], c3 = ctr[4 * i + 3];
    cwc_philox10(c0, c1, c2, c3, rk);
    out[4 * i] = c0;
    out[4 * i + 1] = c1;
    out[4 * i + 2] = c2;
    out[4 * i + 3] = c3;
}

__global__ void k_log(int64_t n, const double* x, double* out, const cwc_logtab_entry* tab) {
    __shared__ __align__(16) cwc_logsmem s;
    cwc_logsmem_init(s, tab);
    __syncthreads();
    int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
    if (i < n) out[i] = cwc_log(x[i], s);
}

__global__ void k_u01(int64_t n, const uint32_t* w, double* out) {
    __shared__ __align__(16) cwc_logsmem s;
    if (threadIdx.x == 0) s.k[6] = 0x1.fffffffffffffp-1;  // the constant cwc_logsmem_init stores
    __syncthreads();
    int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
    if (i < n) out[i] = cwc_u01(w[2 * i], w[2 * i + 1], s.k[6]);
}

__global__ void k_div(int64_t n, const double* num, const double* den, double* out) {
    int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
    if (i < n) out[i] = cwc_div(num[i], den[i]);
}

void ck(cudaError_t e, const char* what) {
    if (e != cudaSuccess) throw cwc::Error(CWC_E_CUDA, std::string(what) + ": " + cudaGetErrorString(e));
}

template <class T>
T* dev_copy(const T* h, size_t n) {
    T* d = nullptr;
    ck(cudaMalloc(&d, n * sizeof(T) + 16), "cudaMalloc");
    if (h) ck(cudaMemcpy(d, h, n * sizeof(T), cudaMemcpyHostToDevice), "H2D");
    return d;
}

}  // namespace

namespace cwc {

void selftest_philox(int64_t n, const uint32_t* ctr, const uint32_t* key, uint32_t* out) {
    if (n <= 0) return;
    uint32_t *dc = dev_copy(ctr, 4 * n), *dk = dev_copy(key, 2 * n), *dout = dev_copy<uint32_t>(nullptr, 4 * n);
    k_philox<<<(unsigned)((n + 255) / 256), 256>>>(n, dc, dk, dout);
    ck(cudaGetLastError(), "k_philox");
    ck(cudaMemcpy(out, dout, 4 * n * sizeof(uint32_t), cudaMemcpyDeviceToHost), "D2H");
    cudaFree(dc); cudaFree(dk); cudaFree(dout);
}

void selftest_log(int64_t n, const double* x, double* out) {
    if (n <= 0) return;
    cwc_logtab_entry tab[128];
    build_log_table(tab);
    cwc_logtab_entry* dt = dev_copy(tab, 128);
    double *dx = dev_copy(x, n), *dout = dev_copy<double>(nullptr, n);
    k_log<<<(unsigned)((n + 255) / 256), 256>>>(n, dx, dout, dt);
    ck(cudaGetLastError(), "k_log");
    ck(cudaMemcpy(out, dout, n * sizeof(double), cudaMemcpyDeviceToHost), "D2H");
    cudaFree(dt); cudaFree(dx); cudaFree(dout);
}

void selftest_div(int64_t n, const double* num, const double* den, double* out) {
    if (n <= 0) return;
    double *dn = dev_copy(num, n), *dd = dev_copy(den, n), *dout = dev_copy<double>(nullptr, n);
    k_div<<<(unsigned)((n + 255) / 256), 256>>>(n, dn, dd, dout);
    ck(cudaGetLastError(), "k_div");
    ck(cudaMemcpy(out, dout, n * sizeof(double), cudaMemcpyDeviceToHost), "D2H");
    cudaFree(dn); cudaFree(dd); cudaFree(dout);
}

void selftest_u01(int64_t n, const uint32_t* words, double* out) {
    if (n <= 0) return;
    uint32_t* dw = dev_copy(words, 2 * n);
    double* dout = dev_copy<double>(nullptr, n);
    k_u01<<<(unsigned)((n + 255) / 256), 256>>>(n, dw, dout);
    ck(cudaGetLastError(), "k_u01");
    ck(cudaMemcpy(out, dout, n * sizeof(double), cudaMemcpyDeviceToHost), "D2H");
    cudaFree(dw); cudaFree(dout);
}

}  // namespace cwc

// Microbenchmark (development aid): dependent-chain latency and single-SMSP reciprocal throughput
// of the SASS operations the SSA step is made of (the latency table of tools/sched_sim.py).
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/lat_micro tools/lat_micro.cu
// One block of 32 threads (one warp on one SMSP); clock64 around an unrolled chain; the
// instruction mix is checked with cuobjdump -sass.
#include <cstdio>
#include <cuda_runtime.h>

#define N 256

#define CHAIN(name, T, init, body)                                                \
    __global__ void name(long long* cyc, T* out, T seed) {                        \
        T x = init;                                                               \
        long long t0 = clock64();                                                 \
        _Pragma("unroll") for (int i = 0; i < N; ++i) { body; }                   \
        long long t1 = clock64();                                                 \
        out[threadIdx.x] = x;                                                     \
        if (threadIdx.x == 0) cyc[0] = t1 - t0;                                   \
    }

CHAIN(k_dadd, double, seed + threadIdx.x, asm volatile("add.rn.f64 %0, %0, %1;" : "+d"(x) : "d"(seed)))
CHAIN(k_dmul, double, seed + threadIdx.x, asm volatile("mul.rn.f64 %0, %0, %1;" : "+d"(x) : "d"(seed)))
CHAIN(k_dfma, double, seed + threadIdx.x, asm volatile("fma.rn.f64 %0, %0, %1, %1;" : "+d"(x) : "d"(seed)))
CHAIN(k_rcp, double, seed + threadIdx.x, asm volatile("rcp.approx.ftz.f64 %0, %0;" : "+d"(x)))
CHAIN(k_lop3, unsigned, seed + threadIdx.x,
      asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(x) : "r"(seed), "r"(seed * 3u)))
CHAIN(k_iadd3, unsigned, seed + threadIdx.x, asm volatile("add.u32 %0, %0, %1;" : "+r"(x) : "r"(seed)))
CHAIN(k_imad, unsigned, seed + threadIdx.x, asm volatile("mad.lo.u32 %0, %0, %1, %1;" : "+r"(x) : "r"(seed)))
CHAIN(k_imadhi, unsigned, seed + threadIdx.x, asm volatile("mul.hi.u32 %0, %0, %1;" : "+r"(x) : "r"(seed | 1u)))
// IMAD.WIDE.U32 + LOP3 (hi ^ lo feeds the next multiply; subtract the LOP3 latency)
CHAIN(k_imadwide, unsigned, seed + threadIdx.x, {
    unsigned long long p;
    asm volatile("mul.wide.u32 %0, %1, %2;" : "=l"(p) : "r"(x), "r"(0xD2511F53u));
    x = (unsigned)p ^ (unsigned)(p >> 32);
})
// I2F.F64: int -> double, the double's high word feeds the next conversion
CHAIN(k_i2f64, int, (int)(seed + threadIdx.x), {
    double d;
    asm volatile("cvt.rn.f64.s32 %0, %1;" : "=d"(d) : "r"(x));
    x = __double2hiint(d);
})
CHAIN(k_dsetp_sel, double, seed + threadIdx.x, {
    double y;
    asm volatile("{.reg .pred p; setp.lt.f64 p, %1, %2; selp.f64 %0, %1, %2, p;}" : "=d"(y) : "d"(x), "d"(seed));
    x = y;
})

__global__ void k_lds(long long* cyc, int* out, int seed) {
    __shared__ int s[1024];
    for (int i = threadIdx.x; i < 1024; i += 32) s[i] = (i * 7 + 1) & 1023;
    __syncwarp();
    int x = seed & 1023;
    long long t0 = clock64();
#pragma unroll
    for (int i = 0; i < N; ++i) x = s[x];
    long long t1 = clock64();
    out[threadIdx.x] = x;
    if (threadIdx.x == 0) cyc[0] = t1 - t0;
}

// reciprocal throughput: 8 independent chains in one warp
#define TPUT(name, T, body)                                                       \
    __global__ void name(long long* cyc, T* out, T seed) {                        \
        T x[8];                                                                   \
        _Pragma("unroll") for (int j = 0; j < 8; ++j) x[j] = seed + threadIdx.x + j; \
        long long t0 = clock64();                                                 \
        _Pragma("unroll") for (int i = 0; i < N / 8; ++i) {                       \
            _Pragma("unroll") for (int j = 0; j < 8; ++j) { body; }               \
        }                                                                         \
        long long t1 = clock64();                                                 \
        T s = 0;                                                                  \
        _Pragma("unroll") for (int j = 0; j < 8; ++j) s += x[j];                  \
        out[threadIdx.x] = s;                                                     \
        if (threadIdx.x == 0) cyc[0] = t1 - t0;                                   \
    }

TPUT(t_dfma, double, asm volatile("fma.rn.f64 %0, %0, %1, %1;" : "+d"(x[j]) : "d"(seed)))
TPUT(t_lop3, unsigned, asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(x[j]) : "r"(seed), "r"(seed * 3u)))
TPUT(t_imad, unsigned, asm volatile("mad.lo.u32 %0, %0, %1, %1;" : "+r"(x[j]) : "r"(seed)))
TPUT(t_imadwide, unsigned, {
    unsigned long long p;
    asm volatile("mul.wide.u32 %0, %1, %2;" : "=l"(p) : "r"(x[j]), "r"(0xD2511F53u));
    x[j] = (unsigned)p ^ (unsigned)(p >> 32);
})
TPUT(t_i2f64, int, {
    double d;
    asm volatile("cvt.rn.f64.s32 %0, %1;" : "=d"(d) : "r"(x[j]));
    x[j] = __double2hiint(d);
})
TPUT(t_rcp, double, asm volatile("rcp.approx.ftz.f64 %0, %0;" : "+d"(x[j])))

template <class K, class T>
double run(K k, T seed) {
    long long* c;
    T* o;
    cudaMalloc(&c, 8);
    cudaMalloc(&o, 32 * sizeof(T));
    long long h = 0;
    for (int rep = 0; rep < 3; ++rep) {
        k<<<1, 32>>>(c, o, seed);
        cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    }
    cudaFree(c);
    cudaFree(o);
    return (double)h / N;
}

// ---- pipe sharing: two independent op kinds interleaved, 8 chains each (cycles per pair)
#define MIX(name, T1, T2, body1, body2)                                           \
    __global__ void name(long long* cyc, double* out, double seed) {              \
        T1 a[8];                                                                  \
        T2 b[8];                                                                  \
        _Pragma("unroll") for (int j = 0; j < 8; ++j) {                           \
            a[j] = (T1)(seed + threadIdx.x + j);                                  \
            b[j] = (T2)(seed * 3 + threadIdx.x + j);                              \
        }                                                                         \
        long long t0 = clock64();                                                 \
        _Pragma("unroll") for (int i = 0; i < N / 8; ++i) {                       \
            _Pragma("unroll") for (int j = 0; j < 8; ++j) { body1; body2; }       \
        }                                                                         \
        long long t1 = clock64();                                                 \
        double s = 0;                                                             \
        _Pragma("unroll") for (int j = 0; j < 8; ++j) s += (double)a[j] + (double)b[j]; \
        out[blockIdx.x * blockDim.x + threadIdx.x] = s;                           \
        if (threadIdx.x == 0) cyc[0] = t1 - t0;                                   \
    }
// IMAD.WIDE + LOP3 (the Philox round pattern): 2 instructions
#define B_WIDE(v) { unsigned long long p_; asm volatile("mul.wide.u32 %0, %1, %2;" : "=l"(p_) : "r"(v), "r"(0xD2511F53u)); \
                    v = (unsigned)p_ ^ (unsigned)(p_ >> 32); }
#define B_DFMA(v) asm volatile("fma.rn.f64 %0, %0, %0, %0;" : "+d"(v))
#define B_LOP3(v) asm volatile("lop3.b32 %0, %0, %0, 7, 0x96;" : "+r"(v))
#define B_IMAD(v) asm volatile("mad.lo.u32 %0, %0, %0, 7;" : "+r"(v))
#define B_I2F(v) { double d_; asm volatile("cvt.rn.f64.s32 %0, %1;" : "=d"(d_) : "r"(v)); v = __double2hiint(d_); }
MIX(m_wide_only, unsigned, unsigned, B_WIDE(a[j]), B_WIDE(b[j]))
MIX(m_wide_dfma, unsigned, double, B_WIDE(a[j]), B_DFMA(b[j]))
MIX(m_wide_lop3, unsigned, unsigned, B_WIDE(a[j]), B_LOP3(b[j]))
MIX(m_wide_imad, unsigned, unsigned, B_WIDE(a[j]), B_IMAD(b[j]))
MIX(m_dfma_only, double, double, B_DFMA(a[j]), B_DFMA(b[j]))
MIX(m_dfma_imad, double, unsigned, B_DFMA(a[j]), B_IMAD(b[j]))
MIX(m_dfma_lop3, double, unsigned, B_DFMA(a[j]), B_LOP3(b[j]))
MIX(m_imad_lop3, unsigned, unsigned, B_IMAD(a[j]), B_LOP3(b[j]))
MIX(m_dfma_i2f, double, int, B_DFMA(a[j]), B_I2F(b[j]))

// warps = 1: one SMSP; 4: one warp per SMSP (all four busy); 8: two per SMSP (cycles per pair per warp)
template <class K>
double run_mix(K k, int warps) {
    long long* c;
    double* o;
    cudaMalloc(&c, 8);
    cudaMalloc(&o, 32 * warps * sizeof(double));
    long long h = 0;
    for (int rep = 0; rep < 3; ++rep) {
        k<<<1, 32 * warps>>>(c, o, 1.25);
        cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    }
    cudaFree(c);
    cudaFree(o);
    return (double)h / N;
}

void main_mix() {
    printf("pipe sharing (cycles per pair of independent ops, wide = IMAD.WIDE+LOP3; 1 warp | 4 warps = 1 per SMSP | 8 warps):\n");
#define R(k) printf("  %-14s %.2f | %.2f | %.2f\n", #k, run_mix(k, 1), run_mix(k, 4), run_mix(k, 8))
    R(m_wide_only);
    R(m_wide_dfma);
    R(m_wide_lop3);
    R(m_wide_imad);
    R(m_dfma_only);
    R(m_dfma_imad);
    R(m_dfma_lop3);
    R(m_imad_lop3);
    R(m_dfma_i2f);
}

int main() {
    printf("latency (cycles, dependent chain, 1 warp):\n");
    printf("  DADD        %.2f\n", run(k_dadd, 1.000001));
    printf("  DMUL        %.2f\n", run(k_dmul, 1.000001));
    printf("  DFMA        %.2f\n", run(k_dfma, 0.5));
    printf("  MUFU.RCP64H %.2f\n", run(k_rcp, 1.5));
    printf("  LOP3        %.2f\n", run(k_lop3, 7u));
    printf("  IADD        %.2f\n", run(k_iadd3, 7u));
    printf("  IMAD        %.2f\n", run(k_imad, 7u));
    printf("  IMAD.HI     %.2f\n", run(k_imadhi, 7u));
    printf("  IMAD.WIDE+LOP3 %.2f\n", run(k_imadwide, 7u));
    printf("  I2F.F64     %.2f\n", run(k_i2f64, 7));
    printf("  DSETP+SEL   %.2f\n", run(k_dsetp_sel, 0.5));
    printf("  LDS         %.2f\n", run(k_lds, 7));
    printf("reciprocal throughput (cycles per warp-instruction, 8 chains, 1 warp):\n");
    printf("  DFMA        %.2f\n", run(t_dfma, 0.5));
    printf("  LOP3        %.2f\n", run(t_lop3, 7u));
    printf("  IMAD        %.2f\n", run(t_imad, 7u));
    printf("  IMAD.WIDE+LOP3 %.2f (2 instr)\n", run(t_imadwide, 7u));
    printf("  I2F.F64     %.2f\n", run(t_i2f64, 7));
    printf("  MUFU.RCP64H %.2f\n", run(t_rcp, 1.5));
    main_mix();
    return 0;
}

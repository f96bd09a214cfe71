// Issue-rate microbenchmarks for the instructions the two hot paths are built from
// (FADD/FMUL, packed FADD2/FMUL2, VABSDIFF4.U8.ACC, PRMT, SHFL) on sm_100a.
// Prints ops per clock per SM. Run: ./ubench
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
#include <cstdlib>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { printf("CUDA %s @%d\n", cudaGetErrorString(e), __LINE__); return 1; } } while (0)

constexpr int ITERS = 4096;
constexpr int CH = 8;  // independent chains per thread

__device__ unsigned long long g_sink;
__device__ long long g_cyc[4096];

__device__ __forceinline__ unsigned long long f2add(unsigned long long a, unsigned long long b) {
  unsigned long long d; asm volatile("add.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b)); return d;
}
__device__ __forceinline__ unsigned long long f2mul(unsigned long long a, unsigned long long b) {
  unsigned long long d; asm volatile("mul.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b)); return d;
}

template <int KIND>
__global__ void __launch_bounds__(256, 4) kbench(float seedf, unsigned seedu) {
  long long t0 = clock64();
  float f[CH]; unsigned u[CH]; unsigned long long p[CH];
  #pragma unroll
  for (int c = 0; c < CH; ++c) {
    f[c] = seedf + c + threadIdx.x; u[c] = seedu * (c + 1) + threadIdx.x;
    p[c] = ((unsigned long long)__float_as_uint(f[c]) << 32) | __float_as_uint(f[c] + 1.f);
  }
  const float w = 0.33333334f;
  const unsigned long long w2 = ((unsigned long long)__float_as_uint(w) << 32) | __float_as_uint(w);
  const unsigned long long mzr = (unsigned long long)seedu << 63 | ((unsigned long long)seedu << 31);
  for (int it = 0; it < ITERS; ++it) {
    #pragma unroll
    for (int c = 0; c < CH; ++c) {
      if (KIND == 0) {          // FADD reg,reg
        f[c] = __fadd_rn(f[c], f[(c + 1) % CH]);
      } else if (KIND == 1) {   // FMUL by constant
        f[c] = __fmul_rn(f[c], w);
      } else if (KIND == 2) {   // FADD2 (packed f32x2)
        p[c] = f2add(p[c], p[(c + 1) % CH]);
      } else if (KIND == 3) {   // FMUL2 packed by packed constant
        p[c] = f2mul(p[c], w2);
      } else if (KIND == 4) {   // VABSDIFF4 with accumulate
        u[c] = __vsadu4(u[(c + 3) % CH], seedu + c) + u[c];
      } else if (KIND == 5) {   // raw vabsdiff4 PTX with add (single instr)
        unsigned d; asm volatile("vabsdiff4.u32.u32.u32.add %0, %1, %2, %3;" : "=r"(d) : "r"(u[(c + 3) % CH]), "r"(seedu ^ c), "r"(u[c])); u[c] = d;
      } else if (KIND == 6) {   // PRMT
        u[c] = __byte_perm(u[c], u[(c + 1) % CH], 0x4321 + c);
      } else if (KIND == 7) {   // SHFL
        u[c] = __shfl_up_sync(0xffffffffu, u[c], 1) + c;
      } else if (KIND == 8) {   // Jacobi update unpacked: ((a+b)+c)*w  (3 FP ops)
        f[c] = __fmul_rn(__fadd_rn(__fadd_rn(f[c], f[(c + 1) % CH]), f[(c + 2) % CH]), w);
      } else if (KIND == 9) {   // Jacobi update packed f32x2 (3 FP2 ops = 6 flops)
        p[c] = f2mul(f2add(f2add(p[c], p[(c + 1) % CH]), p[(c + 2) % CH]), w2);
      } else if (KIND == 11) {  // Jacobi packed exactly as the kernel: FADD2, FADD2, FFMA2(x, w, -0 reg)
        unsigned long long d;
        asm volatile("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(d) : "l"(f2add(f2add(p[c], p[(c + 1) % CH]), p[(c + 2) % CH])), "l"(w2), "l"(mzr));
        p[c] = d;
      } else if (KIND == 10) {  // mixed: VABSDIFF4 + FADD in parallel pipes
        unsigned d; asm volatile("vabsdiff4.u32.u32.u32.add %0, %1, %2, %3;" : "=r"(d) : "r"(u[(c + 3) % CH]), "r"(seedu ^ c), "r"(u[c])); u[c] = d;
        f[c] = __fadd_rn(f[c], f[(c + 1) % CH]);
      }
    }
  }
  long long t1 = clock64();
  unsigned long long s = 0;
  #pragma unroll
  for (int c = 0; c < CH; ++c) s += __float_as_uint(f[c]) + u[c] + p[c];
  if (s == 0x1234567ull) g_sink = s;
  if (threadIdx.x == 0) g_cyc[blockIdx.x] = t1 - t0;
}

template <int KIND>
int run(const char* name, double ops_per_inner, int blocks) {
  kbench<KIND><<<blocks, 256>>>(1.0f, 7u);
  CK(cudaDeviceSynchronize());
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  cudaEventRecord(a);
  kbench<KIND><<<blocks, 256>>>(1.0f, 7u);
  cudaEventRecord(b);
  CK(cudaDeviceSynchronize());
  float ms; cudaEventElapsedTime(&ms, a, b);
  static long long cyc[4096];
  CK(cudaMemcpyFromSymbol(cyc, g_cyc, sizeof(long long) * blocks));
  long long mx = 0; double mean = 0;
  for (int i = 0; i < blocks; ++i) { if (cyc[i] > mx) mx = cyc[i]; mean += cyc[i]; }
  mean /= blocks;
  int nsm; cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
  double thread_ops = (double)blocks * 256 * ITERS * CH * ops_per_inner;
  double per_sm_clk = thread_ops / nsm / (double)mx;
  double ghz = (double)mx / (ms * 1e6);
  printf("%-28s  %8.1f thread-ops/clk/SM  (max cyc %lld, mean %.0f, %.3f ms, implied clk %.3f GHz, %.3e ops/s)\n",
         name, per_sm_clk, mx, mean, ms, ghz, thread_ops / (ms * 1e-3));
  return 0;
}

int main(int argc, char** argv) {
  int nsm; cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
  cudaDeviceProp pr; cudaGetDeviceProperties(&pr, 0);
  printf("device %s  SMs %d  smem/SM %zu  regs/SM %d  cc %d.%d\n", pr.name, nsm, pr.sharedMemPerMultiprocessor, pr.regsPerMultiprocessor, pr.major, pr.minor);
  int blocks = nsm * (argc > 1 ? atoi(argv[1]) : 4);  // one resident wave (4 x 256 threads/SM)
  run<0>("FADD r,r", 1, blocks);
  run<1>("FMUL r,imm", 1, blocks);
  run<2>("FADD2 (x2 flops)", 2, blocks);
  run<3>("FMUL2 (x2 flops)", 2, blocks);
  run<4>("__vsadu4 + add (bytes)", 4, blocks);
  run<5>("vabsdiff4.add (bytes)", 4, blocks);
  run<6>("PRMT", 1, blocks);
  run<7>("SHFL (+IADD)", 1, blocks);
  run<8>("jacobi unpacked (updates)", 1, blocks);
  run<9>("jacobi f32x2 (updates)", 2, blocks);
  run<10>("vabsdiff4 bytes (+FADD mix)", 4, blocks);
  run<11>("jacobi f32x2 as kernel (upd)", 2, blocks);
  return 0;
}

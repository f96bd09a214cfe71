// Isolate 2-D/3-D tensor TMA loads of uint8 frames (box origin at arbitrary / negative
// byte offsets).  ./tma_probe <variant>: 0 = 2D driver-linked, 1 = 3D driver-linked,
// 2 = 3D via cudaGetDriverEntryPoint, 3 = 3D + prefetch.tensormap
#include <cuda.h>
#include <cuda_runtime.h>
#include <cstdio>
#include <cstdint>
#include <cstdlib>
#include <vector>

__device__ __forceinline__ uint32_t sa(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }

template <int DIM, bool PF>
__global__ void k(const __grid_constant__ CUtensorMap m, int x, int y, uint8_t* out, int nbytes) {
  extern __shared__ __align__(128) uint8_t raw[];
  uint8_t* s = (uint8_t*)(((uintptr_t)raw + 127) & ~(uintptr_t)127);
  __shared__ __align__(8) uint64_t bar;
  if (threadIdx.x == 0) {
    if (PF) asm volatile("prefetch.tensormap [%0];" :: "l"(&m) : "memory");
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" :: "r"(sa(&bar)));
    asm volatile("fence.mbarrier_init.release.cluster;");
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" :: "r"(sa(&bar)), "r"(nbytes));
    if (DIM == 2)
      asm volatile("cp.async.bulk.tensor.2d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3}], [%4];"
                   :: "r"(sa(s)), "l"(&m), "r"(x), "r"(y), "r"(sa(&bar)) : "memory");
    else
      asm volatile("cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];"
                   :: "r"(sa(s)), "l"(&m), "r"(x), "r"(y), "r"(0), "r"(sa(&bar)) : "memory");
  }
  __syncthreads();
  asm volatile("{\n\t.reg .pred p;\n\tW: mbarrier.try_wait.parity.shared::cta.b64 p, [%0], 0;\n\t@!p bra W;\n\t}" :: "r"(sa(&bar)) : "memory");
  for (int i = threadIdx.x; i < nbytes; i += blockDim.x) out[i] = s[i];
}

typedef CUresult (*Enc)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*, const cuuint64_t*,
                        const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave, CUtensorMapSwizzle,
                        CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

int main(int argc, char** argv) {
  int v = argc > 1 ? atoi(argv[1]) : 0;
  const int W = 64, H = 48, B = 48;
  std::vector<uint8_t> h(W * H);
  for (int i = 0; i < W * H; ++i) h[i] = (uint8_t)(i * 7 + 3);
  uint8_t *d, *o;
  cudaMalloc(&d, W * H); cudaMalloc(&o, B * B);
  cudaMemcpy(d, h.data(), W * H, cudaMemcpyHostToDevice);
  Enc enc = nullptr;
  if (v == 2 || v == 3) {
    void* p; cudaDriverEntryPointQueryResult q;
    cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q);
    enc = (Enc)p;
  } else {
    enc = (Enc)cuTensorMapEncodeTiled;
  }
  CUtensorMap m;
  int dim = (v == 0 || v >= 4) ? 2 : 3;
  cuuint64_t dims[3] = {W, H, 1};
  cuuint64_t str[2] = {W, (cuuint64_t)W * H};
  cuuint32_t box[3] = {B, B, 1};
  cuuint32_t es[3] = {1, 1, 1};
  int x = -13, y = -5;
  CUtensorMapL2promotion l2 = CU_TENSOR_MAP_L2_PROMOTION_L2_128B;
  if (v == 4) { x = 0; y = 0; }
  if (v == 5) { x = 16; y = 0; box[0] = 16; box[1] = 16; }
  if (v == 6) { x = 0; y = 0; l2 = CU_TENSOR_MAP_L2_PROMOTION_NONE; }
  if (v == 7) { x = 0; y = 0; box[0] = 64; box[1] = 32; }
  if (v == 8) { x = 3; y = 0; }
  if (v == 9) { x = -16; y = 0; }
  if (v == 10) { x = 0; y = -5; }
  if (v == 11) { x = 5; y = 7; box[0] = 16; box[1] = 8; }
  if (v == 12) { x = 17; y = 0; box[0] = 32; box[1] = 8; }
  CUresult r = enc(&m, CU_TENSOR_MAP_DATA_TYPE_UINT8, dim, d, dims, str, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                   CU_TENSOR_MAP_SWIZZLE_NONE, l2, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  printf("variant %d encode %d\n", v, (int)r);
  const int nb = box[0] * box[1];
  if (v == 0 || v >= 4) k<2, false><<<1, 128, B * B + 128>>>(m, x, y, o, nb);
  else if (v == 3) k<3, true><<<1, 128, B * B + 128>>>(m, x, y, o, nb);
  else k<3, false><<<1, 128, B * B + 128>>>(m, x, y, o, nb);
  cudaError_t e = cudaDeviceSynchronize();
  printf("variant %d kernel: %s\n", v, cudaGetErrorString(e));
  std::vector<uint8_t> g(B * B);
  cudaMemcpy(g.data(), o, B * B, cudaMemcpyDeviceToHost);
  int bad = 0;
  for (int yy = 0; yy < (int)box[1]; ++yy) for (int xx = 0; xx < (int)box[0]; ++xx) {
    int gx = x + xx, gy = y + yy;
    uint8_t want = (gx >= 0 && gx < W && gy >= 0 && gy < H) ? h[gy * W + gx] : 0;
    bad += g[yy * box[0] + xx] != want;
  }
  printf("variant %d mismatches %d\n", v, bad);
  return 0;
}

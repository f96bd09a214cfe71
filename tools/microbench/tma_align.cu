// Does a tiled (SWIZZLE_NONE) cp.async.bulk.tensor accept a shared-memory destination that is
// 16-byte but not 128-byte aligned?  Loads a 48 x 48 uint8 box to offsets 0, 16, 32, 48, 96 and
// checks the bytes.  Build: nvcc -gencode arch=compute_100a,code=sm_100a -I<csrc> tma_align.cu -o tma_align
#include <cuda.h>
#include <cuda_runtime.h>
#include <cstdio>
#include <cstdlib>
#include <cstdint>
#include <vector>
#include "sm100_ptx.cuh"
using namespace sp::ptx;

typedef CUresult (*EncodeTiledFn)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                  const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                  CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

__global__ void k(const __grid_constant__ CUtensorMap map, int off, int x, int y, uint8_t* out) {
    extern __shared__ __align__(128) uint8_t sm[];
    __shared__ __align__(8) uint64_t bar;
    uint8_t* base = sm + ((128u - (smem_addr(sm) & 127u)) & 127u);
    if (threadIdx.x == 0) {
        mbar_init(&bar, 1);
        fence_mbar_init();
        mbar_arrive_expect_tx(&bar, 48 * 48);
        tma_load_3d(base + off, &map, x, y, 0, &bar);
    }
    __syncthreads();
    mbar_wait(&bar, 0);
    for (int i = threadIdx.x; i < 48 * 48; i += blockDim.x) out[i] = base[off + i];
}

int main(int argc, char** argv) {
    const int W = 256, H = 128;
    std::vector<uint8_t> h(W * H);
    for (int i = 0; i < W * H; ++i) h[i] = (uint8_t)(i * 7 + (i / W) * 13);
    uint8_t *d, *o;
    cudaMalloc(&d, W * H);
    cudaMalloc(&o, 48 * 48);
    cudaMemcpy(d, h.data(), W * H, cudaMemcpyHostToDevice);
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q);
    EncodeTiledFn enc = (EncodeTiledFn)p;
    CUtensorMap m;
    cuuint64_t dims[3] = {(cuuint64_t)W, (cuuint64_t)H, 1};
    cuuint64_t strides[2] = {(cuuint64_t)W, (cuuint64_t)W * H};
    cuuint32_t box[3] = {48, 48, 1}, es[3] = {1, 1, 1};
    CUresult r = enc(&m, CU_TENSOR_MAP_DATA_TYPE_UINT8, 3, d, dims, strides, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                     CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_128B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    printf("encode %d\n", (int)r);
    const int off = atoi(argv[1]), x = atoi(argv[2]);
    {
            k<<<1, 128, 8192>>>(m, off, x, 3, o);
            cudaError_t e = cudaDeviceSynchronize();
            if (e != cudaSuccess) {
                printf("off %d x %d: %s\n", off, x, cudaGetErrorString(e));
                return 1;
            }
            std::vector<uint8_t> g(48 * 48);
            cudaMemcpy(g.data(), o, 48 * 48, cudaMemcpyDeviceToHost);
            int bad = 0;
            for (int r2 = 0; r2 < 48; ++r2)
                for (int c = 0; c < 48; ++c) {
                    int gx = x + c, gy = 3 + r2;
                    uint8_t want = (gx >= 0 && gx < W && gy < H) ? h[gy * W + gx] : 0;
                    bad += g[r2 * 48 + c] != want;
                }
            printf("off %3d x %3d: %s (%d bad)\n", off, x, bad ? "WRONG" : "ok", bad);
    }
    return 0;
}

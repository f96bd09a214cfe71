// ablation.cu — SURVEY §8(f) row N1: the paper's "GPU w/o scratchpad memory" baselines
// (the staged kernels were 8x (ME) and 10x (Jacobi) faster than versions that
// "use only GPU DRAM"; Figs. 4-5 "GPU Perf w/o Scratchpad memory").  Same arithmetic, same
// results (bit-exact), no explicitly managed on-chip staging and no time tiling:
//   * sp_jacobi1d_untiled   — one launch per time step, every operand read from global
//     memory (each step streams the whole array through HBM: 8 B per point-update);
//   * sp_me_sad_search_direct — one CTA per macroblock, one thread per candidate at a
//     time, every pixel read from global memory (through L1/L2 only).
#include <cuda_runtime.h>

#include <cstdint>

#include "../../include/sp.h"
#include "sm100_ptx.cuh"
#include "sp_internal.h"

namespace {

constexpr float kWf = 0.333333343267440796f;  // fl32(1/3) = 0x3EAAAAAB

__global__ void __launch_bounds__(256) jacobi_step_direct(const float* __restrict__ src, float* __restrict__ dst,
                                                          int64_t n) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        if (i == 0 || i == n - 1) {
            dst[i] = src[i];
        } else {
            const float s = __fadd_rn(__fadd_rn(src[i - 1], src[i]), src[i + 1]);
            dst[i] = __fmul_rn(s, kWf);
        }
    }
}

__device__ __forceinline__ uint64_t key_of(uint32_t s, int dx, int dy, int R) {
    const uint32_t l1 = (uint32_t)(abs(dx) + abs(dy));
    return ((uint64_t)s << 21) | ((uint64_t)l1 << 14) | ((uint64_t)(dy + R) << 7) | (uint64_t)(dx + R);
}

__global__ void __launch_bounds__(128) me_direct_kernel(const uint8_t* __restrict__ ref, const uint8_t* __restrict__ cur,
                                                        int64_t pitch, int32_t width, int32_t frame_height,
                                                        int32_t row0, int64_t pair_stride, int32_t R,
                                                        int32_t mb_row_begin, int32_t mb_rows, int16_t* mv,
                                                        uint32_t* best, uint32_t* surface) {
    __shared__ uint64_t wkeys[4];
    const int bx = blockIdx.x, byr = blockIdx.y, pair = blockIdx.z;
    const int mbx = gridDim.x;
    const int x0 = 16 * bx, y0 = 16 * (mb_row_begin + byr);
    const uint8_t* rp = ref + (int64_t)pair * pair_stride;
    const uint8_t* cp = cur + (int64_t)pair * pair_stride;
    const int side = 2 * R + 1;
    const size_t mb_index = ((size_t)pair * mb_rows + byr) * mbx + bx;
    uint64_t bestk = ~0ull;
    for (int c = threadIdx.x; c < side * side; c += blockDim.x) {
        const int dy = c / side - R, dx = c % side - R;
        const bool valid = (x0 + dx >= 0) && (x0 + dx + 16 <= width) && (y0 + dy >= 0) && (y0 + dy + 16 <= frame_height);
        uint32_t a = 0xffffffffu;
        if (valid) {
            a = 0;
            const int xs = x0 + dx, sh = 8 * (xs & 3);
            for (int v = 0; v < 16; ++v) {
                const uint32_t* cw = reinterpret_cast<const uint32_t*>(cp + (int64_t)(y0 + v - row0) * pitch + x0);
                const uint32_t* rw =
                    reinterpret_cast<const uint32_t*>(rp + (int64_t)(y0 + dy + v - row0) * pitch + (xs & ~3));
                uint32_t w[5];
#pragma unroll
                for (int k = 0; k < 4; ++k) w[k] = rw[k];
                w[4] = sh ? rw[4] : 0u;
#pragma unroll
                for (int k = 0; k < 4; ++k) a = sp::ptx::sad4(__funnelshift_r(w[k], w[k + 1], sh), cw[k], a);
            }
            const uint64_t k = key_of(a, dx, dy, R);
            bestk = k < bestk ? k : bestk;
        }
        if (surface) surface[mb_index * side * side + c] = a;
    }
    for (int o = 16; o; o >>= 1) {
        const uint64_t other = __shfl_xor_sync(0xffffffffu, bestk, o);
        bestk = other < bestk ? other : bestk;
    }
    if ((threadIdx.x & 31) == 0) wkeys[threadIdx.x >> 5] = bestk;
    __syncthreads();
    if (threadIdx.x == 0) {
        uint64_t b = wkeys[0];
        for (int w = 1; w < (int)(blockDim.x >> 5); ++w) b = wkeys[w] < b ? wkeys[w] : b;
        mv[2 * mb_index] = (int16_t)((int)(b & 127) - R);
        mv[2 * mb_index + 1] = (int16_t)((int)((b >> 7) & 127) - R);
        best[mb_index] = (uint32_t)(b >> 21);
    }
}

}  // namespace

extern "C" int sp_jacobi1d_untiled(float* a, float* work, int64_t n, int32_t steps, void* stream) {
    SP_NVTX("sp_jacobi1d_untiled");
    if (!a || !work || a == work || n < 3 || steps < 0) return SP_ERR_INVALID_ARG;
    const cudaStream_t s = (cudaStream_t)stream;
    float* cur = a;
    float* nxt = work;
    const int64_t blocks64 = (n + 255) / 256;
    const int blocks = (int)(blocks64 < 148 * 64 ? blocks64 : 148 * 64);
    for (int32_t t = 0; t < steps; ++t) {
        jacobi_step_direct<<<blocks, 256, 0, s>>>(cur, nxt, n);
        float* tmp = cur;
        cur = nxt;
        nxt = tmp;
    }
    SP_CUDA_TRY(cudaGetLastError());
    if (cur != a) SP_CUDA_TRY(cudaMemcpyAsync(a, cur, (size_t)n * sizeof(float), cudaMemcpyDeviceToDevice, s));
    return SP_OK;
}

extern "C" int sp_me_sad_search_direct(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                                       int32_t rows_in_buffer, int32_t row0_global, int32_t frame_height,
                                       int32_t n_pairs, int64_t pair_stride, int32_t block, int32_t range,
                                       int32_t mb_row_begin, int32_t mb_row_end, int16_t* mv, uint32_t* best_sad,
                                       uint32_t* surface, void* stream) {
    SP_NVTX("sp_me_sad_search_direct");
    if (block != 16) return SP_ERR_UNSUPPORTED;
    if (!ref || !cur || !mv || !best_sad || range < 0 || range > 63 || width < 16 || frame_height < 16 ||
        n_pairs < 0 || rows_in_buffer < 1 || (pitch & 3) || pitch < width || (reinterpret_cast<uintptr_t>(ref) & 3) ||
        (reinterpret_cast<uintptr_t>(cur) & 3) || (n_pairs > 1 && (pair_stride & 3)))
        return SP_ERR_INVALID_ARG;
    const int mbx = width / 16, mby = frame_height / 16;
    if (mb_row_begin < 0 || mb_row_end > mby || mb_row_begin > mb_row_end) return SP_ERR_INVALID_ARG;
    const int rows = mb_row_end - mb_row_begin;
    if (n_pairs == 0 || rows == 0) return SP_OK;
    me_direct_kernel<<<dim3(mbx, rows, n_pairs), 128, 0, (cudaStream_t)stream>>>(
        ref, cur, pitch, width, frame_height, row0_global, n_pairs > 1 ? pair_stride : 0, range, mb_row_begin, rows,
        mv, best_sad, surface);
    SP_CUDA_TRY(cudaGetLastError());
    return SP_OK;
}

// me.cu — full-search SAD motion estimation on sm_100a (SURVEY §8(a) rows H1, H3, H4,
// H5b, H6, H7).
//
// The paper's Fig. 2 nest: FORALL search positions (i, j) x FOR pixels
// (k, l) < WS = 16, tiled over thread blocks and threads (Fig. 3; the paper's
// 8800 GTX run used 32 blocks x 256 threads, tiles (32,16,16,16)).  On B200:
//   * one CTA per macroblock (outer tile); threads own register tiles of 4 x 8
//     candidates (4 dx values of one byte phase x 8 consecutive dy values);
//   * move-in (H4): the macroblock's reference window — the Alg. 2 bounding box
//     [y0-R, y0+15+R] x [x0-R, x0+15+R] of ref[y0+dy+v][x0+dx+u] (H3) — is staged by
//     the TMA unit (3-D tensor map, out-of-frame pixels zero-filled — their candidates
//     are invalid anyway), then expanded on chip into FOUR byte-phase copies (column
//     origin x0-R+p, p = 0..3; one funnel shift per word, ~2% of the ALU work) so every
//     candidate row is a run of 4-byte-aligned words and the SAD loop executes no byte
//     permute (the TMA box origin itself must be 16-byte aligned, probe: tools/probes);
//     the current macroblock is staged once and hoisted into 64 registers (§4.2 hoisting,
//     `cur` does not depend on the candidate loops);
//   * compute (H5b): per candidate row, 4 VABSDIFF4.U8.ACC (4 pixels + accumulate each);
//     each loaded window row feeds up to 8 dy candidates x 4 dx candidates in registers;
//   * argmin (H6, fused): lexicographic (SAD, |dx|+|dy|, dy, dx) as a 64-bit key,
//     reduced in-thread, then across the warp with two CREDUX.MIN, then across warps;
//   * move-out (H7): MV (int16 x 2) + SAD (u32) per macroblock, optional full surface.
// The candidates dx = +R (column) and dy = +R (row) fall outside the 2R x 2R register
// tiling; they are swept by a per-candidate loop over the same staged copies.
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdint>
#include <mutex>

#include "../../include/sp.h"
#include "sm100_ptx.cuh"
#include "sp_internal.h"

namespace {

using namespace sp::ptx;

constexpr int kMB = 16;      // macroblock edge (WS = 16)
constexpr int kTy = 8;       // dy candidates per thread
constexpr int kTx = 4;       // dx candidates per thread (same byte phase, stride 4)
constexpr int kRows = kTy + kMB - 1;  // window rows a thread sweeps (23)

struct MeArgs {
    int32_t width, frame_height, row0, range;
    int32_t mbx, mb_row_begin, mb_rows;
    int32_t win;  // window edge = 2R + 16 (bytes per copy row, rows per copy)
    int16_t* mv;
    uint32_t* sad;
    uint32_t* surface;
};

__device__ __forceinline__ uint64_t make_key(uint32_t s, int dx, int dy, int R) {
    const uint32_t l1 = (uint32_t)(abs(dx) + abs(dy));
    return ((uint64_t)s << 21) | ((uint64_t)l1 << 14) | ((uint64_t)(dy + R) << 7) | (uint64_t)(dx + R);
}

// Warp-wide minimum of a 64-bit key with two 32-bit CREDUX.MIN.
__device__ __forceinline__ uint64_t warp_min_key(uint64_t k) {
    const uint32_t hi = (uint32_t)(k >> 32), lo = (uint32_t)k;
    const uint32_t mh = __reduce_min_sync(0xffffffffu, hi);
    const uint32_t ml = __reduce_min_sync(0xffffffffu, hi == mh ? lo : 0xffffffffu);
    return ((uint64_t)mh << 32) | ml;
}

// Fast path: R in {16, 32} (x0 - R 16-byte aligned); blockDim = R*R/8.
__global__ void __launch_bounds__(128, 3)
me_sad_kernel(const __grid_constant__ CUtensorMap ref_map, const __grid_constant__ CUtensorMap cur_map, MeArgs A) {
    extern __shared__ __align__(128) uint8_t smem_raw[];
    __shared__ __align__(8) uint64_t bar;
    __shared__ uint64_t warp_keys[32];
    // TMA tile destinations must be 128-byte aligned
    uint8_t* smem = reinterpret_cast<uint8_t*>((reinterpret_cast<uintptr_t>(smem_raw) + 127) & ~uintptr_t(127));

    const int R = A.range;
    const int win = A.win;
    const int copy_bytes = win * win;
    uint8_t* cur_s = smem + 4 * copy_bytes;
    const int tid = threadIdx.x, nthr = blockDim.x;
    const int bx = blockIdx.x, byr = blockIdx.y, pair = blockIdx.z;
    const int by = A.mb_row_begin + byr;  // global MB row
    const int x0 = kMB * bx, y0 = kMB * by;
    const int ywin = y0 - R - A.row0;  // buffer row of window row 0

    if (tid == 0) {
        prefetch_tmap(&ref_map);
        prefetch_tmap(&cur_map);
        mbar_init(&bar, 1);
        fence_mbar_init();
        mbar_arrive_expect_tx(&bar, (uint32_t)(copy_bytes + kMB * kMB));
        // the TMA box origin must be 16-byte aligned in the innermost dimension, so the
        // window is staged once at x0 - R (R % 16 == 0) and the byte phases are built below
        tma_load_3d(smem, &ref_map, x0 - R, ywin, pair, &bar);
        tma_load_3d(cur_s, &cur_map, x0, y0 - A.row0, pair, &bar);
    }
    __syncthreads();
    mbar_wait(&bar, 0);
    {   // byte-phase copies p = 1..3: word q of copy p = bytes [4q+p, 4q+p+4) of the row
        const int v4_per_row = win / 16;
        const int nv4 = win * v4_per_row;
        for (int v = tid; v < nv4; v += nthr) {
            const int r = v / v4_per_row, c = v - r * v4_per_row;
            const uint32_t* row = reinterpret_cast<const uint32_t*>(smem + r * win);
            const uint4 w = reinterpret_cast<const uint4*>(row)[c];
            const uint32_t nx = (c + 1 < v4_per_row) ? row[4 * c + 4] : 0u;
#pragma unroll
            for (int p = 1; p < 4; ++p) {
                uint4 o;
                o.x = __funnelshift_r(w.x, w.y, 8 * p);
                o.y = __funnelshift_r(w.y, w.z, 8 * p);
                o.z = __funnelshift_r(w.z, w.w, 8 * p);
                o.w = __funnelshift_r(w.w, nx, 8 * p);
                reinterpret_cast<uint4*>(smem + p * copy_bytes + r * win)[c] = o;
            }
        }
    }
    __syncthreads();

    // hoisted current block: 16 rows x 4 words
    uint32_t C[kMB][4];
#pragma unroll
    for (int v = 0; v < kMB; ++v) {
        const uint4 q = reinterpret_cast<const uint4*>(cur_s)[v];
        C[v][0] = q.x;
        C[v][1] = q.y;
        C[v][2] = q.z;
        C[v][3] = q.w;
    }

    const int ngx = R / 8;             // dx groups per phase
    const int nmain = ngx * 4 * (R / 4);
    uint64_t best = ~0ull;
    const int side = 2 * R + 1;
    const int W = A.width, Hf = A.frame_height;
    const size_t mb_index = ((size_t)pair * A.mb_rows + byr) * A.mbx + bx;

    if (tid < nmain) {
        const int p = tid & 3;
        const int g = (tid >> 2) % ngx;
        const int d = tid / (4 * ngx);
        uint32_t acc[kTx][kTy];
#pragma unroll
        for (int j = 0; j < kTx; ++j)
#pragma unroll
            for (int i = 0; i < kTy; ++i) acc[j][i] = 0;
        const uint8_t* rowp = smem + p * copy_bytes + (kTy * d) * win + 16 * g;
#pragma unroll
        for (int r = 0; r < kRows; ++r) {
            const uint4 w0 = *reinterpret_cast<const uint4*>(rowp + r * win);
            const uint4 w1 = *reinterpret_cast<const uint4*>(rowp + r * win + 16);
            const uint32_t Wd[8] = {w0.x, w0.y, w0.z, w0.w, w1.x, w1.y, w1.z, w1.w};
#pragma unroll
            for (int i = 0; i < kTy; ++i) {
                const int v = r - i;
                if (v < 0 || v >= kMB) continue;
#pragma unroll
                for (int j = 0; j < kTx; ++j) {
                    uint32_t a = acc[j][i];
                    a = sad4(Wd[j + 0], C[v][0], a);
                    a = sad4(Wd[j + 1], C[v][1], a);
                    a = sad4(Wd[j + 2], C[v][2], a);
                    a = sad4(Wd[j + 3], C[v][3], a);
                    acc[j][i] = a;
                }
            }
        }
        // epilogue: validity, keys, optional surface
        const bool interior = (x0 - R >= 0) && (x0 + 16 + R <= W) && (y0 - R >= 0) && (y0 + 16 + R <= Hf);
#pragma unroll
        for (int j = 0; j < kTx; ++j) {
            const int dx = -R + p + 4 * (4 * g + j);
#pragma unroll
            for (int i = 0; i < kTy; ++i) {
                const int dy = -R + kTy * d + i;
                const bool valid =
                    interior || ((x0 + dx >= 0) && (x0 + dx + 16 <= W) && (y0 + dy >= 0) && (y0 + dy + 16 <= Hf));
                const uint64_t k = valid ? make_key(acc[j][i], dx, dy, R) : ~0ull;
                best = k < best ? k : best;
                if (A.surface) A.surface[mb_index * side * side + (size_t)(dy + R) * side + (dx + R)] = valid ? acc[j][i] : 0xffffffffu;
            }
        }
    }
    // tail candidates: column dx = +R (dy in [-R, R]) and row dy = +R (dx in [-R, R-1])
    const int ntail = 4 * R + 1;
    for (int c = tid; c < ntail; c += nthr) {
        int dx, dy;
        if (c < side) {
            dx = R;
            dy = -R + c;
        } else {
            dx = -R + (c - side);
            dy = R;
        }
        const int p = (dx + R) & 3, m = (dx + R) >> 2;
        const uint32_t* rw = reinterpret_cast<const uint32_t*>(smem + p * copy_bytes + (dy + R) * win) + m;
        uint32_t a = 0;
#pragma unroll
        for (int v = 0; v < kMB; ++v) {
            const uint32_t* q = rw + v * (win / 4);
            a = sad4(q[0], C[v][0], a);
            a = sad4(q[1], C[v][1], a);
            a = sad4(q[2], C[v][2], a);
            a = sad4(q[3], C[v][3], a);
        }
        const bool valid = (x0 + dx >= 0) && (x0 + dx + 16 <= W) && (y0 + dy >= 0) && (y0 + dy + 16 <= Hf);
        const uint64_t k = valid ? make_key(a, dx, dy, R) : ~0ull;
        best = k < best ? k : best;
        if (A.surface) A.surface[mb_index * side * side + (size_t)(dy + R) * side + (dx + R)] = valid ? a : 0xffffffffu;
    }
    // argmin across the CTA
    best = warp_min_key(best);
    const int warp = tid >> 5, lane = tid & 31, nwarps = (nthr + 31) >> 5;
    if (lane == 0) warp_keys[warp] = best;
    __syncthreads();
    if (tid == 0) {
        uint64_t b = warp_keys[0];
        for (int w = 1; w < nwarps; ++w) b = warp_keys[w] < b ? warp_keys[w] : b;
        const int dx = (int)(b & 127) - R, dy = (int)((b >> 7) & 127) - R;
        A.mv[2 * mb_index] = (int16_t)dx;
        A.mv[2 * mb_index + 1] = (int16_t)dy;
        A.sad[mb_index] = (uint32_t)(b >> 21);
    }
}

// Generic path (any 0 <= R <= 63): window staged byte-wise with zero fill, one thread per
// candidate at a time.  Used for ranges outside the fast path's envelope.
__global__ void __launch_bounds__(256) me_sad_generic_kernel(const uint8_t* __restrict__ ref,
                                                             const uint8_t* __restrict__ cur, int64_t pitch,
                                                             int32_t rows_in_buffer, int64_t pair_stride, MeArgs A) {
    extern __shared__ __align__(16) uint8_t smem[];
    __shared__ uint64_t warp_keys[32];
    const int R = A.range, win = A.win;
    uint8_t* win_s = smem;
    uint8_t* cur_s = smem + win * win;
    const int tid = threadIdx.x, nthr = blockDim.x;
    const int bx = blockIdx.x, byr = blockIdx.y, pair = blockIdx.z;
    const int by = A.mb_row_begin + byr;
    const int x0 = kMB * bx, y0 = kMB * by;
    const uint8_t* rp = ref + (int64_t)pair * pair_stride;
    const uint8_t* cp = cur + (int64_t)pair * pair_stride;
    for (int q = tid; q < win * win; q += nthr) {
        const int wy = q / win, wx = q % win;
        const int gy = y0 - R + wy - A.row0, gx = x0 - R + wx;
        uint8_t v = 0;
        if (gy >= 0 && gy < rows_in_buffer && gx >= 0 && gx < A.width) v = rp[(int64_t)gy * pitch + gx];
        win_s[q] = v;
    }
    for (int q = tid; q < kMB * kMB; q += nthr) cur_s[q] = cp[(int64_t)(y0 - A.row0 + q / kMB) * pitch + x0 + q % kMB];
    __syncthreads();
    const int side = 2 * R + 1;
    const size_t mb_index = ((size_t)pair * A.mb_rows + byr) * A.mbx + bx;
    uint64_t best = ~0ull;
    for (int c = tid; c < side * side; c += nthr) {
        const int dy = c / side - R, dx = c % side - R;
        uint32_t a = 0;
        for (int v = 0; v < kMB; ++v)
            for (int u = 0; u < kMB; ++u) {
                const int x = cur_s[v * kMB + u], y = win_s[(dy + R + v) * win + (dx + R + u)];
                a += (uint32_t)(x > y ? x - y : y - x);
            }
        const bool valid = (x0 + dx >= 0) && (x0 + dx + 16 <= A.width) && (y0 + dy >= 0) && (y0 + dy + 16 <= A.frame_height);
        const uint64_t k = valid ? make_key(a, dx, dy, R) : ~0ull;
        best = k < best ? k : best;
        if (A.surface) A.surface[mb_index * side * side + c] = valid ? a : 0xffffffffu;
    }
    best = warp_min_key(best);
    if ((tid & 31) == 0) warp_keys[tid >> 5] = best;
    __syncthreads();
    if (tid == 0) {
        uint64_t b = warp_keys[0];
        for (int w = 1; w < (nthr + 31) / 32; ++w) b = warp_keys[w] < b ? warp_keys[w] : b;
        A.mv[2 * mb_index] = (int16_t)((int)(b & 127) - R);
        A.mv[2 * mb_index + 1] = (int16_t)((int)((b >> 7) & 127) - R);
        A.sad[mb_index] = (uint32_t)(b >> 21);
    }
}

// ---- tensor maps through the driver entry point (no libcuda link dependency) ----------
typedef CUresult (*EncodeTiledFn)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                  const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                  CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

EncodeTiledFn get_encode() {
    static EncodeTiledFn fn = nullptr;
    static std::once_flag once;
    std::call_once(once, [] {
        void* p = nullptr;
        cudaDriverEntryPointQueryResult q;
        if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
            q == cudaDriverEntryPointSuccess)
            fn = reinterpret_cast<EncodeTiledFn>(p);
    });
    return fn;
}

int make_map(CUtensorMap* m, const uint8_t* base, int32_t width, int32_t rows, int32_t n_pairs, int64_t pitch,
             int64_t pair_stride, uint32_t box_w, uint32_t box_h) {
    EncodeTiledFn enc = get_encode();
    if (!enc) {
        sp::set_cuda_error((int)cudaErrorNotSupported);
        return SP_ERR_CUDA;
    }
    cuuint64_t dims[3] = {(cuuint64_t)width, (cuuint64_t)rows, (cuuint64_t)n_pairs};
    cuuint64_t strides[2] = {(cuuint64_t)pitch, (cuuint64_t)pair_stride};
    cuuint32_t box[3] = {box_w, box_h, 1};
    cuuint32_t estr[3] = {1, 1, 1};
    CUresult r = enc(m, CU_TENSOR_MAP_DATA_TYPE_UINT8, 3, const_cast<uint8_t*>(base), dims, strides, box, estr,
                     CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_128B,
                     CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (r != CUDA_SUCCESS) {
        sp::set_cuda_error((int)r);
        return SP_ERR_CUDA;
    }
    return SP_OK;
}

bool fast_range(int R) { return R == 16 || R == 32; }

}  // namespace

extern "C" int sp_me_ref_window(int32_t width, int32_t frame_height, int32_t range, int32_t bx, int32_t by,
                                int64_t lb[2], int64_t ub[2]) {
    if (!lb || !ub || width < kMB || frame_height < kMB || range < 0 || bx < 0 || by < 0 || bx >= width / kMB ||
        by >= frame_height / kMB)
        return SP_ERR_INVALID_ARG;
    const int64_t x0 = (int64_t)kMB * bx, y0 = (int64_t)kMB * by;
    lb[0] = y0 - range > 0 ? y0 - range : 0;
    lb[1] = x0 - range > 0 ? x0 - range : 0;
    ub[0] = y0 + kMB - 1 + range < frame_height - 1 ? y0 + kMB - 1 + range : frame_height - 1;
    ub[1] = x0 + kMB - 1 + range < width - 1 ? x0 + kMB - 1 + range : width - 1;
    return SP_OK;
}

extern "C" int sp_me_sad_search(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                                int32_t rows_in_buffer, int32_t row0_global, int32_t frame_height, int32_t n_pairs,
                                int64_t pair_stride, int32_t block, int32_t range, int32_t mb_row_begin,
                                int32_t mb_row_end, int16_t* mv, uint32_t* best_sad, uint32_t* surface, void* stream) {
    if (block != kMB) return SP_ERR_UNSUPPORTED;
    if (!ref || !cur || !mv || !best_sad) return SP_ERR_INVALID_ARG;
    if (range < 0 || range > 63 || width < kMB || frame_height < kMB || n_pairs < 0 || rows_in_buffer < 1)
        return SP_ERR_INVALID_ARG;
    if (pitch < width || (pitch & 15) || (pair_stride & 15) || (reinterpret_cast<uintptr_t>(ref) & 15) ||
        (reinterpret_cast<uintptr_t>(cur) & 15))
        return SP_ERR_INVALID_ARG;
    if (n_pairs > 1 && pair_stride < pitch * rows_in_buffer) return SP_ERR_INVALID_ARG;
    const int mbx = width / kMB, mby = frame_height / kMB;
    if (mb_row_begin < 0 || mb_row_end > mby || mb_row_begin > mb_row_end) return SP_ERR_INVALID_ARG;
    // the band must hold every row the current blocks of these MB rows occupy
    if (mb_row_end > mb_row_begin &&
        (row0_global > kMB * mb_row_begin || row0_global + rows_in_buffer < kMB * mb_row_end))
        return SP_ERR_INVALID_ARG;
    const int rows = mb_row_end - mb_row_begin;
    if (n_pairs == 0 || rows == 0 || mbx == 0) return SP_OK;
    const cudaStream_t s = (cudaStream_t)stream;
    MeArgs a{width, frame_height, row0_global, range, mbx, mb_row_begin, rows, 2 * range + 16, mv, best_sad, surface};
    dim3 grid(mbx, rows, n_pairs);
    if (fast_range(range)) {
        CUtensorMap rm, cm;
        int st;
        if ((st = make_map(&rm, ref, width, rows_in_buffer, n_pairs, pitch, n_pairs > 1 ? pair_stride : pitch * rows_in_buffer,
                           (uint32_t)a.win, (uint32_t)a.win)))
            return st;
        if ((st = make_map(&cm, cur, width, rows_in_buffer, n_pairs, pitch, n_pairs > 1 ? pair_stride : pitch * rows_in_buffer,
                           kMB, kMB)))
            return st;
        const int smem = 4 * a.win * a.win + kMB * kMB + 128;
        static std::once_flag once;
        static cudaError_t attr_err = cudaSuccess;
        std::call_once(once, [] {
            attr_err = cudaFuncSetAttribute(me_sad_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 4 * 80 * 80 + 256 + 128);
        });
        SP_CUDA_TRY(attr_err);
        const int threads = ((range * range / 8) + 31) & ~31;
        me_sad_kernel<<<grid, threads, smem, s>>>(rm, cm, a);
    } else {
        const int smem = a.win * a.win + kMB * kMB;
        static std::once_flag once;
        static cudaError_t attr_err = cudaSuccess;
        std::call_once(once, [] {
            attr_err = cudaFuncSetAttribute(me_sad_generic_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 142 * 142 + 256);
        });
        SP_CUDA_TRY(attr_err);
        me_sad_generic_kernel<<<grid, 256, smem, s>>>(ref, cur, pitch, rows_in_buffer, n_pairs > 1 ? pair_stride : 0, a);
    }
    SP_CUDA_TRY(cudaGetLastError());
    return SP_OK;
}

// jacobi.cu — time-tiled 1-D Jacobi on sm_100a.
//
// The paper's method (Fig. 3) on B200:
//   * one kernel launch = one time tile ("pass") of h <= Tt steps; the launch boundary is
//     the global synchronisation between time tiles (row H8);
//   * outer tiles (S owned cells) -> persistent CTAs, taken in sequence (the paper's
//     memory-limit sub-tiles run one after another inside an outer-level process,
//     P:L627-637); warps own 2*32*K-cell strips (inner tiles -> threads);
//   * move-in (H4): each tile's footprint — the Alg. 2 bounding box
//     [x0-H, x0+S-1+H] ∩ [0, n-1] (H3) — is staged into shared memory by a 1-D TMA bulk
//     copy, double-buffered so the next tile streams in while this one computes;
//   * compute (H5a): each thread holds 2K cells in registers as K packed fp32 pairs
//     (u_j, v_j) = (cell l*K+j, cell 32K+l*K+j of its warp's strip) so that every update
//     is half of one FADD2/FADD2/FMUL2 triple; lane neighbours come from warp shuffles;
//     warp strips overlap by H cells on each side, so h steps need no barrier at all
//     (overlapped "concurrent start" tiling, reading R-J4);
//   * move-out (H7): only owned cells, at the final step (reading R-J5), registers ->
//     shared memory -> coalesced 128-bit global stores.
// Arithmetic is b = ((a[i-1] + a[i]) + a[i+1]) * w, each op rounded to nearest fp32, never
// contracted (PTX add.rn/mul.rn), w = fl32(1/3) — bit-identical to the definition.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <mutex>

#include "../../include/sp.h"
#include "sm100_ptx.cuh"
#include "sp_internal.h"

namespace {

using namespace sp::ptx;

constexpr int kK = 16;                   // packed pairs per thread
constexpr int kWarps = 8;                // warps per CTA
constexpr int kThreads = 32 * kWarps;    // 256
constexpr int kStrip = 64 * kK;          // cells per warp strip (1024)
constexpr int kStage = kWarps * kStrip;  // floats per shared-memory stage (8192 = 32 KB)
constexpr int kStages = 2;
constexpr int kMaxTimeTile = 128;
constexpr uint32_t kW = 0x3EAAAAABu;  // fl32(1/3)
constexpr uint64_t kNegZero2 = 0x8000000080000000ull;

struct PassArgs {
    const float* src;  // src[j] holds global cell g0 + j
    float* dst;        // same indexing
    int64_t n;         // global cells
    int64_t g0, len;   // available window of src
    int64_t own_begin, own_end;  // owned cells written to dst (global indices)
    int64_t S;         // owned cells per tile
    int64_t tiles;
    int32_t h;         // steps in this pass
    int32_t H;         // staged halo (multiple of 4, >= h)
    int32_t wo;        // owned cells per warp (multiple of 4)
    int64_t* flog;     // nullable: [tiles][2] footprint of this pass
    uint64_t mz;       // (-0.0f, -0.0f), opaque to ptxas (see f2_mul_nofuse)
};

// One Jacobi step on the thread's 2K cells.  kBoundary: the warp strip contains global
// cell 0 or n-1, which must keep its value (fix_u / fix_v: bit j set = pair j's u / v
// component is a fixed boundary cell).
template <bool kBoundary>
__device__ __forceinline__ void step(uint64_t (&P)[kK], int lane, uint64_t w2, uint64_t mz, uint32_t fix_u, uint32_t fix_v) {
    const float ul = f2_lo(P[kK - 1]), vl = f2_hi(P[kK - 1]);
    const float uf = f2_lo(P[0]), vf = f2_hi(P[0]);
    const float a = __shfl_sync(0xffffffffu, ul, (lane + 31) & 31);  // lane-1's last u
    const float b = __shfl_sync(0xffffffffu, vl, (lane + 31) & 31);  // lane-1's last v
    const float c = __shfl_sync(0xffffffffu, uf, (lane + 1) & 31);   // lane+1's first u
    const float d = __shfl_sync(0xffffffffu, vf, (lane + 1) & 31);   // lane+1's first v
    // the v strip continues the u strip: lane 0's v-left is lane 31's last u and
    // lane 31's u-right is lane 0's first v
    uint64_t prev = f2_pack(a, lane == 0 ? a : b);
    const uint64_t right = f2_pack(lane == 31 ? d : c, d);
#pragma unroll
    for (int j = 0; j < kK; ++j) {
        const uint64_t cur = P[j];
        const uint64_t nxt = (j + 1 < kK) ? P[j + 1] : right;
        uint64_t r = f2_mul_nofuse(f2_add(f2_add(prev, cur), nxt), w2, mz);
        if (kBoundary) {
            if ((fix_u >> j) & 1u) r = f2_pack(f2_lo(cur), f2_hi(r));
            if ((fix_v >> j) & 1u) r = f2_pack(f2_lo(r), f2_hi(cur));
        }
        P[j] = r;
        prev = cur;
    }
}

__global__ void __launch_bounds__(kThreads, 3) jacobi1d_pass_kernel(PassArgs A) {
    extern __shared__ __align__(128) float smem[];
    __shared__ __align__(8) uint64_t full[kStages];

    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const uint64_t w2 = (uint64_t(kW) << 32) | kW;
    const int64_t G = gridDim.x;
    const int64_t first = blockIdx.x;

    const int64_t lo_avail = A.g0 > 0 ? A.g0 : 0;
    const int64_t hi_avail = (A.g0 + A.len < A.n) ? A.g0 + A.len : A.n;

    // Footprint actually transferred for tile t: [lo, hi) with lo 16-byte aligned; the
    // 16-byte-multiple prefix goes by TMA, a <= 3-cell ragged end by plain loads.
    auto tile_range = [&](int64_t t, int64_t& x0, int64_t& st, int64_t& lo, int64_t& hi) {
        x0 = A.own_begin + t * A.S;
        st = A.own_end - x0 < A.S ? A.own_end - x0 : A.S;
        lo = x0 - A.H > lo_avail ? x0 - A.H : lo_avail;
        hi = x0 + st + A.H < hi_avail ? x0 + st + A.H : hi_avail;
    };
    auto issue = [&](int64_t t, int s) {  // single thread
        int64_t x0, st, lo, hi;
        tile_range(t, x0, st, lo, hi);
        const uint32_t bytes = (uint32_t)(((hi - lo) & ~int64_t(3)) * 4);
        mbar_arrive_expect_tx(&full[s], bytes);
        if (bytes) tma_load_1d(smem + s * kStage + (lo - (x0 - A.H)), A.src + (lo - A.g0), bytes, &full[s]);
    };

    if (tid == 0) {
        for (int s = 0; s < kStages; ++s) mbar_init(&full[s], 1);
        fence_mbar_init();
    }
    __syncthreads();
    if (tid == 0) {
        for (int s = 0; s < kStages; ++s)
            if (first + s * G < A.tiles) issue(first + s * G, s);
    }

    int it = 0;
    for (int64_t t = first; t < A.tiles; t += G, ++it) {
        const int s = it & 1;
        const uint32_t parity = (it >> 1) & 1;
        float* buf = smem + s * kStage;
        int64_t x0, st, lo, hi;
        tile_range(t, x0, st, lo, hi);
        const int64_t base = x0 - A.H;  // buf[j] <-> global base + j
        {   // ragged end (<= 3 cells) that the 16-byte TMA could not carry
            const int64_t tail0 = lo + ((hi - lo) & ~int64_t(3));
            if (tid < hi - tail0) buf[tail0 - base + tid] = A.src[tail0 + tid - A.g0];
        }
        if (tid == 0 && A.flog) {
            const int64_t flb = x0 - A.h > 0 ? x0 - A.h : 0;
            const int64_t fub = x0 + st - 1 + A.h < A.n - 1 ? x0 + st - 1 + A.h : A.n - 1;
            A.flog[2 * t] = flb;
            A.flog[2 * t + 1] = fub;
        }
        mbar_wait(&full[s], parity);
        __syncthreads();  // ragged-end stores visible

        // ---- registers <- staged strip -------------------------------------------------
        const int wofs = warp * A.wo;                 // strip start in buf (multiple of 4)
        const int64_t rb = base + wofs;               // global index of strip cell 0
        uint64_t P[kK];
        {
            const float4* pu = reinterpret_cast<const float4*>(buf + wofs + lane * kK);
            const float4* pv = reinterpret_cast<const float4*>(buf + wofs + 32 * kK + lane * kK);
#pragma unroll
            for (int q = 0; q < kK / 4; ++q) {
                const float4 u = pu[q], v = pv[q];
                P[4 * q + 0] = f2_pack(u.x, v.x);
                P[4 * q + 1] = f2_pack(u.y, v.y);
                P[4 * q + 2] = f2_pack(u.z, v.z);
                P[4 * q + 3] = f2_pack(u.w, v.w);
            }
        }
        // ---- h steps in registers ---------------------------------------------------
        const bool boundary = (rb <= 0 && 0 < rb + kStrip) || (rb <= A.n - 1 && A.n - 1 < rb + kStrip);
        if (!boundary) {
            for (int k = 0; k < A.h; ++k) step<false>(P, lane, w2, A.mz, 0u, 0u);
        } else {
            const int64_t cu = rb + lane * kK, cv = rb + 32 * kK + lane * kK;
            uint32_t fix_u = 0, fix_v = 0;
            if (cu <= 0 && 0 < cu + kK) fix_u |= 1u << (0 - cu);
            if (cu <= A.n - 1 && A.n - 1 < cu + kK) fix_u |= 1u << (A.n - 1 - cu);
            if (cv <= 0 && 0 < cv + kK) fix_v |= 1u << (0 - cv);
            if (cv <= A.n - 1 && A.n - 1 < cv + kK) fix_v |= 1u << (A.n - 1 - cv);
            for (int k = 0; k < A.h; ++k) step<true>(P, lane, w2, A.mz, fix_u, fix_v);
        }
        __syncthreads();  // every warp has finished reading this stage

        // ---- owned cells -> staged buffer (move-out staging) -------------------------
        {
            // warp owns strip offsets [H, H + own_w); tile-local owned range is [H, H + st)
            const int own_lo = A.H;
            const int64_t rem_w = st - (int64_t)wofs;
            const int own_hi = A.H + (int)(rem_w < A.wo ? rem_w : (int64_t)A.wo);
            float4* qu = reinterpret_cast<float4*>(buf + wofs + lane * kK);
            float4* qv = reinterpret_cast<float4*>(buf + wofs + 32 * kK + lane * kK);
#pragma unroll
            for (int q = 0; q < kK / 4; ++q) {
                const int ou = lane * kK + 4 * q, ov = 32 * kK + lane * kK + 4 * q;
                if (ou >= own_lo && ou < own_hi)
                    qu[q] = make_float4(f2_lo(P[4 * q]), f2_lo(P[4 * q + 1]), f2_lo(P[4 * q + 2]), f2_lo(P[4 * q + 3]));
                if (ov >= own_lo && ov < own_hi)
                    qv[q] = make_float4(f2_hi(P[4 * q]), f2_hi(P[4 * q + 1]), f2_hi(P[4 * q + 2]), f2_hi(P[4 * q + 3]));
            }
        }
        __syncthreads();
        // ---- coalesced 128-bit copy of the owned cells to global ----------------------
        {
            const float4* s4 = reinterpret_cast<const float4*>(buf + A.H);
            float4* d4 = reinterpret_cast<float4*>(A.dst + (x0 - A.g0));
            const int n4 = (int)(st >> 2);
            for (int q = tid; q < n4; q += kThreads) d4[q] = s4[q];
            const int rem = (int)(st & 3);
            if (tid < rem) A.dst[x0 - A.g0 + 4 * n4 + tid] = buf[A.H + 4 * n4 + tid];
        }
        fence_proxy_async_smem();
        __syncthreads();  // stage free: refill it with tile t + 2G
        if (tid == 0 && t + 2 * G < A.tiles) issue(t + 2 * G, s);
    }
}

struct DeviceInfo {
    int sms = 0;
    int occ = 0;
    bool ok = false;
};

int device_info(DeviceInfo& out) {
    static std::mutex mu;
    static DeviceInfo cache[64];
    int dev = 0;
    SP_CUDA_TRY(cudaGetDevice(&dev));
    std::lock_guard<std::mutex> lk(mu);
    DeviceInfo& d = cache[dev & 63];
    if (!d.ok) {
        SP_CUDA_TRY(cudaDeviceGetAttribute(&d.sms, cudaDevAttrMultiProcessorCount, dev));
        const int smem = kStages * kStage * (int)sizeof(float);
        SP_CUDA_TRY(cudaFuncSetAttribute(jacobi1d_pass_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, smem));
        SP_CUDA_TRY(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&d.occ, jacobi1d_pass_kernel, kThreads, smem));
        if (d.occ < 1) d.occ = 1;
        d.ok = true;
    }
    out = d;
    return SP_OK;
}

inline int32_t halo_of(int32_t time_tile) { return (time_tile + 3) & ~3; }

int geometry(int32_t time_tile, int32_t space_tile, int64_t& S, int32_t& wo) {
    if (time_tile < 1 || time_tile > kMaxTimeTile) return SP_ERR_INVALID_ARG;
    const int32_t H = halo_of(time_tile);
    const int32_t wo_max = kStrip - 2 * H;  // multiple of 4
    const int64_t S_max = (int64_t)kWarps * wo_max;
    if (space_tile == 0) {
        S = S_max;
        wo = wo_max;
        return SP_OK;
    }
    if (space_tile < 4 || space_tile % 4 != 0 || space_tile > S_max) return SP_ERR_INVALID_ARG;
    S = space_tile;
    wo = (int32_t)(((S + kWarps - 1) / kWarps + 3) & ~int64_t(3));
    return SP_OK;
}

int launch_pass(const PassArgs& a0, cudaStream_t stream, const DeviceInfo& di) {
    PassArgs a = a0;
    if (a.tiles <= 0) return SP_OK;
    const int64_t cap = (int64_t)di.sms * di.occ;
    const int grid = (int)(a.tiles < cap ? a.tiles : cap);
    const int smem = kStages * kStage * (int)sizeof(float);
    jacobi1d_pass_kernel<<<grid, kThreads, smem, stream>>>(a);
    SP_CUDA_TRY(cudaGetLastError());
    return SP_OK;
}

}  // namespace

extern "C" int sp_jacobi1d_plan(int64_t n, int32_t steps, int32_t time_tile, int32_t space_tile, sp_jacobi_plan* out) {
    if (!out || n < 3 || steps < 0) return SP_ERR_INVALID_ARG;
    int64_t S;
    int32_t wo;
    int st = geometry(time_tile, space_tile, S, wo);
    if (st) return st;
    out->n = n;
    out->steps = steps;
    out->time_tile = time_tile;
    out->halo = halo_of(time_tile);
    out->passes = (steps + time_tile - 1) / time_tile;
    out->space_tile = S;
    out->tiles = (n + S - 1) / S;
    out->threads = kThreads;
    out->smem_bytes = kStages * kStage * (int)sizeof(float);
    out->cells_per_thread = 2 * kK;
    DeviceInfo di;
    out->grid = 0;
    if (device_info(di) == SP_OK) {
        const int64_t cap = (int64_t)di.sms * di.occ;
        out->grid = (int32_t)(out->tiles < cap ? out->tiles : cap);
    } else {
        sp::set_cuda_error(0);  // planning works without a device
    }
    return SP_OK;
}

extern "C" int sp_jacobi1d_tile_footprint(int64_t n, int32_t h, int64_t x0, int64_t space_tile, int64_t* lb,
                                          int64_t* ub) {
    if (!lb || !ub || n < 1 || h < 0 || space_tile < 1 || x0 < 0 || x0 >= n) return SP_ERR_INVALID_ARG;
    *lb = x0 - h > 0 ? x0 - h : 0;
    const int64_t e = x0 + space_tile - 1 + h;
    *ub = e < n - 1 ? e : n - 1;
    return SP_OK;
}

extern "C" int sp_jacobi1d_pass_segment(const float* src, float* dst, int64_t n_global, int64_t g0, int64_t len,
                                        int64_t own_begin, int64_t own_end, int32_t h, int32_t time_tile,
                                        int32_t space_tile, void* stream) {
    if (!src || !dst || n_global < 3 || len < 1 || h < 0 || h > time_tile) return SP_ERR_INVALID_ARG;
    if ((reinterpret_cast<uintptr_t>(src) & 15) || (reinterpret_cast<uintptr_t>(dst) & 15)) return SP_ERR_INVALID_ARG;
    if ((g0 & 3) || (own_begin & 3) || own_begin < 0 || own_end > n_global || own_begin > own_end)
        return SP_ERR_INVALID_ARG;
    int64_t S;
    int32_t wo;
    int st = geometry(time_tile, space_tile, S, wo);
    if (st) return st;
    const int32_t H = halo_of(time_tile);
    if (own_begin < g0 || own_end > g0 + len) return SP_ERR_INVALID_ARG;
    if (own_begin - H > 0 && own_begin - H < g0) return SP_ERR_INVALID_ARG;  // halo not available
    if (own_end + H < n_global && own_end + H > g0 + len) return SP_ERR_INVALID_ARG;
    if (h == 0 || own_end == own_begin) {
        if (own_end > own_begin && src != dst)
            SP_CUDA_TRY(cudaMemcpyAsync(dst + (own_begin - g0), src + (own_begin - g0), (own_end - own_begin) * 4,
                                        cudaMemcpyDeviceToDevice, (cudaStream_t)stream));
        return SP_OK;
    }
    DeviceInfo di;
    if ((st = device_info(di))) return st;
    PassArgs a{src, dst, n_global, g0, len, own_begin, own_end, S, (own_end - own_begin + S - 1) / S, h, H, wo, nullptr, kNegZero2};
    return launch_pass(a, (cudaStream_t)stream, di);
}

extern "C" int sp_jacobi1d_timetiled(float* a, float* work, int64_t n, int32_t steps, int32_t time_tile,
                                     int32_t space_tile, int64_t* footprint_log, void* stream) {
    if (!a || !work || n < 3 || steps < 0 || a == work) return SP_ERR_INVALID_ARG;
    if ((reinterpret_cast<uintptr_t>(a) & 15) || (reinterpret_cast<uintptr_t>(work) & 15)) return SP_ERR_INVALID_ARG;
    int64_t S;
    int32_t wo;
    int st = geometry(time_tile, space_tile, S, wo);
    if (st) return st;
    if (steps == 0) return SP_OK;
    DeviceInfo di;
    if ((st = device_info(di))) return st;
    const cudaStream_t s = (cudaStream_t)stream;
    const int32_t H = halo_of(time_tile);
    const int64_t tiles = (n + S - 1) / S;
    float* cur = a;
    float* nxt = work;
    int pass = 0;
    for (int32_t done = 0; done < steps; done += time_tile, ++pass) {
        const int32_t h = steps - done < time_tile ? steps - done : time_tile;
        PassArgs p{cur, nxt, n, 0, n, 0, n, S, tiles, h, H, wo,
                   footprint_log ? footprint_log + (int64_t)pass * tiles * 2 : nullptr, kNegZero2};
        if ((st = launch_pass(p, s, di))) return st;
        float* t = cur;
        cur = nxt;
        nxt = t;
    }
    if (cur != a) SP_CUDA_TRY(cudaMemcpyAsync(a, cur, (size_t)n * sizeof(float), cudaMemcpyDeviceToDevice, s));
    return SP_OK;
}

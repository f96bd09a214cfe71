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
#include <algorithm>
#include <cstdlib>
#include <mutex>
#include <unordered_map>

#include "../../include/sp.h"
#include "sm100_ptx.cuh"
#include "sp_internal.h"

namespace {

using namespace sp::ptx;

constexpr int kMB = 16;      // macroblock edge (WS = 16)
constexpr int kTy = 8;       // dy candidates per thread (R = 32; MeGeom<R>::kTy)
constexpr int kTx = 4;       // dx candidates per thread (same byte phase, stride 4)

#ifndef SP_ME_EXP
#define SP_ME_EXP 0
#endif
// SP_ME_SKIP: a warp whose whole dy band of main candidates is invalid (the first two and the
// last macroblock rows at 1080p, R = 32) runs only its tail candidates: M4 8.368 -> 8.327 ms
// (A/B, r2t).  SP_ME_SCRAMBLE (off): column-major macroblock order, meant to spread those rows
// over the launch, measured slower (8.43 ms).
#ifndef SP_ME_SKIP
#define SP_ME_SKIP 1
#endif
// SP_ME_R16_TY: dy candidates per thread at R = 16.  8 (one warp of 4 x 8 tiles) is the
// default; 4 (two warps of 4 x 4 tiles, 64 registers, 20 warps per SM) measured slower on CIF
// +-16 at throughput: 70.2 vs 72.6 % of the VABSDIFF4 roof (r3d).
#ifndef SP_ME_R16_TY
#define SP_ME_R16_TY 8
#endif
constexpr int sp_me_kTy = 8;
// SP_ME_PHASE_FMA (off): build the byte-phase copies on the FMA pipe (IMAD.HI + IMAD per word)
// instead of the ALU's funnel shift, to unload the binding ALU pipe (the FMA pipe idles at
// ~3 %).  Measured slower (r3y, A/B x 3): M4 8.41-8.48 vs 8.30 ms, CIF +-16 72.0 vs 72.7 % —
// the phase build sits on the path to the CTA barrier, and two dependent multiplies per word
// lengthen it more than the ALU slots they free.
#ifndef SP_ME_PHASE_FMA
#define SP_ME_PHASE_FMA 0
#endif
#ifndef SP_ME_SCRAMBLE
#define SP_ME_SCRAMBLE 0
#endif
#if SP_ME_EXP & 32  // development instrumentation: (smid, start, end) global timer per CTA
__device__ unsigned long long g_me_cta[4096][3];
__device__ __forceinline__ unsigned long long globaltimer() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}
#endif
#if SP_ME_EXP & 16  // development instrumentation: per-section cycle counts per warp
__device__ unsigned long long g_me_prof[8];
#define PMARK(k)                                              \
    do {                                                      \
        const unsigned t_ = (unsigned)clock();                \
        if (lane == 0) prof_s[warp][k] += t_ - t_prev;        \
        t_prev = t_;                                          \
    } while (0)
#else
#define PMARK(k) \
    do {         \
    } while (0)
#endif

// Division of a 32-bit index by a launch constant d >= 1 with a host-computed magic number
// (Granlund-Montgomery, exact for every 32-bit n): one IMAD.HI, two shifts and two adds instead
// of the ~20-instruction reciprocal sequence — the macroblock index -> (pair, row, column)
// split runs on one thread per macroblock, serially in the one-warp R = 16 CTAs.
struct FastDiv {
    uint32_t m, s1, s2;
};
inline FastDiv make_fastdiv(uint32_t d) {
    uint32_t l = 0;
    while (l < 32 && (uint64_t(1) << l) < d) ++l;  // l = ceil(log2 d)
    const uint64_t m = ((uint64_t(1) << 32) * ((uint64_t(1) << l) - d)) / d + 1;
    return FastDiv{(uint32_t)m, l < 1 ? l : 1u, l < 1 ? 0u : l - 1};
}
__device__ __forceinline__ uint32_t fdiv(uint32_t n, const FastDiv& f) {
    const uint32_t t = __umulhi(f.m, n);
    return (t + ((n - t) >> f.s1)) >> f.s2;
}

struct MeArgs {
    int32_t width, frame_height, row0, range, n_pairs;
    int32_t mbx, mb_row_begin, mb_rows;
    int32_t win;  // window edge = 2R + 16 (bytes per copy row, rows per copy)
    int32_t pad;           // frames are edge-extended by `pad` pixels (unrestricted mode), else 0
    int32_t unrestricted;  // 1: every candidate is valid (MVs may point outside the frame)
    int16_t* mv;
    uint32_t* sad;
    uint32_t* surface;
    // nullable: ready[pair] != 0 once both frames of the pair are resident (written by the
    // stream-ordered H2D copies of sp_me_search_host, concurrently with the search); the
    // move-in of a macroblock waits for its pair's flag
    const int32_t* ready;
    // dynamic macroblock distribution: CTA c takes macroblock c first, then the next index
    // from this counter (zero at launch, reset by the last CTA) + gridDim.x.  Co-resident CTAs progress at
    // very different rates (measured: the first of four CTAs on an SM finished after 2.8 ms,
    // the last after 8.8 ms under a static assignment), so static shares left SMs idle.
    uint32_t* counter;
    // Range mode (sp_me_sad_search_range / _gather; 0 otherwise): macroblock mb of the launch is
    // global macroblock mb + flat_mb0 of the (pair, MB row, MB column) space of the whole
    // batch (mb_rows = all MB rows of a frame), outputs are indexed globally, and the tensor
    // maps address pair `pair - pair_base` (the buffer holds frames from pair_base on).
    uint32_t flat_mb0;
    int32_t pair_base;
    uint32_t total_mb;  // macroblocks of this launch (fast kernel)
    uint32_t nrows;     // macroblock rows of this launch (total_mb / mbx)
    FastDiv div_per_pair, div_mbx;  // by mb_rows * mbx and by mbx
    // Class order (R = 16, whole frames, many macroblocks; 0 otherwise): the launch's index
    // space runs over the interior macroblocks of every pair first, then the top / bottom rows,
    // then the left / right columns, then the four corners, so the one code path each class
    // needs (the full search, or a half-frame border search) is the only one the SM's warps run
    // at a time — mixed, the four search loops do not fit the instruction cache together.
    int32_t border_order;
    uint32_t cls_end[3];                 // first index of the rows / columns / corners class
    FastDiv div_int, div_icols, div_rows2, div_cols2;  // by (rows-2)(mbx-2), mbx-2, 2(mbx-2), 2(rows-2)
};

// Fused all-gather of the results over peer memory (sp_me_sad_search_gather): every
// macroblock's (MV, SAD) is stored into the output arrays of every rank (NVLink / CUDA-IPC
// mapped pointers) by the thread that computes it.  Flags: each rank owns u64 flags[2 * nranks]
// = ready[q] (rank q may write into this rank's outputs for epoch e) and done[q] (rank q's
// results of epoch e have all landed here).
constexpr int kMaxGatherRanks = 8;
struct GatherArgs {
    int16_t* mv[kMaxGatherRanks];                 // [q]: rank q's mv array (own one included)
    uint32_t* sad[kMaxGatherRanks];
    unsigned long long* flags[kMaxGatherRanks];  // [q]: rank q's flags (mapped)
    int32_t nranks, rank;
    unsigned long long epoch;
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

// Fast path: R in {16, 32} (x0 - R is then 16-byte aligned, as the TMA box origin must
// be).  Persistent CTAs walk the (pair, MB row, MB column) space with a two-stage pipeline:
// the next macroblock's window and current block stream in by TMA while the current one
// is searched.  Byte-phase copies are double-buffered, so ONE CTA barrier per macroblock
// suffices; the argmin of a macroblock is published by one warp after the next barrier.
template <int R>
struct MeGeom {
    static constexpr int kWin = 2 * R + 16;              // window edge (bytes per row, rows)
    static constexpr int kCopy = kWin * kWin;            // bytes per staged copy (multiple of 128)
    // R = 16: SP_ME_R16_TY dy per thread (8: one warp of 4 x 8 tiles; 4: two warps of 4 x 4)
    static constexpr int kTy = R == 16 ? SP_ME_R16_TY : ::sp_me_kTy;
    static constexpr int kThreads = R * R / kTy;         // one 4 x kTy candidate tile per thread
    static constexpr int kWarps = kThreads / 32;         // 4 (R = 32) or 1 (R = 16)
    static constexpr int kGx = R / 8;                    // dx groups per byte phase
    static constexpr int kTailPer = 4 * R / kThreads;    // tail candidates per thread (+ the corner, split)
    static constexpr int kOffCur = 2 * kCopy;            // cur[2] after raw[2]
    static constexpr int kOffPh = 2 * kCopy + 512;       // phase copies (128-byte aligned)
    // Phase copy slots are kSlot apart and copy ph sits 32*ph bytes into its slot (bank
    // offsets), so a slot must hold kCopy + 96 bytes: with slots only kCopy apart, the last
    // 64 bytes of stage 0's phase-3 copy (window row 2R+15, read by the dy = +R tails) were
    // the first 64 bytes of stage 1's phase-1 copy (row 0), which a warp already building
    // the next macroblock's copies overwrote — a cross-warp race, rare with balanced warps.
    static constexpr int kSlot = kCopy + 128;
    // One-warp CTAs (R = 16) keep ONE set of phase copies: the warp's own __syncwarp orders its
    // compute of macroblock m before its phase build of m + 1, so the second set (which lets
    // 4-warp CTAs get by with one CTA barrier per macroblock) only cost shared memory — 19.8 KB
    // per CTA held the SM to 10 one-warp CTAs (ncu: 9.9 warps active, ALU pipe idle 11 %);
    // 12.5 KB lets the register limit (16 CTAs) bind.
    static constexpr int kPhaseSets = kWarps == 1 ? 1 : 2;
    static constexpr int kSmem = kOffPh + 3 * kPhaseSets * kSlot + 128;  // + alignment slack
    static_assert(kSlot * 3 < 65536 && kOffPh < 65536, "16-bit tail offsets (one-warp CTAs)");
    static_assert(kCopy % 128 == 0, "copies must keep 128-byte alignment");
    static_assert(kSlot >= kCopy + 3 * 32 && kSlot % 128 == 0, "phase copy slots must not overlap");
    static_assert(kWarps == 1 || kWarps == 2 || kWarps == 4, "tail mapping assumes 1, 2 or 4 warps");
    static constexpr int kMinBlocks = kWarps == 4 ? 4 : kWarps == 2 ? 11 : 16;  // CTAs per SM (registers)
    static_assert(kTailPer * kThreads == 4 * R, "tail candidates must spread evenly");
};

// 32-bit argmin key: lexicographic (SAD, |dx|+|dy|, dy, dx) in one unsigned compare.
// Given |dx|+|dy| and dy, |dx| is fixed, so the sign of dx is the only dx information
// left: tie = l1 << 8 | (dy + R) << 1 | (dx > 0) < 2^15 (R <= 32), and
// key = SAD * kKeyMul + tie with kKeyMul = 2^15 + 1 > tie orders exactly like (SAD, tie)
// — a multiplier that is not a power of two keeps the packing on the FMA pipe (IMAD)
// instead of the ALU the SAD instructions need.  Invalid candidates carry SAD =
// kInvalidSad, above every valid SAD (<= 65280) and still without 32-bit overflow.
constexpr uint32_t kKeyMul = 32769u;
constexpr uint32_t kInvalidSad = 0x1FFF0u;
__device__ __forceinline__ uint32_t tie_bits(int dx, int dy, int R) {
    return ((uint32_t)(abs(dx) + abs(dy)) << 8) | ((uint32_t)(dy + R) << 1) | (dx > 0 ? 1u : 0u);
}

// (hi:lo) >> 8 ph for m = 2^(32 - 8 ph), ph in 1..3, on the FMA pipe: lo >> 8 ph = the high word
// of lo * m, hi << (32 - 8 ph) = the low word of hi * m, and the two do not overlap, so one
// multiply-add joins them.  (Inline PTX: the compiler would turn a multiply by a power of two
// back into an ALU shift.)
__device__ __forceinline__ uint32_t shr_bytes_fma(uint32_t lo, uint32_t hi, uint32_t m) {
    uint32_t l, r;
    asm("mul.hi.u32 %0, %1, %2;" : "=r"(l) : "r"(lo), "r"(m));
    asm("mad.lo.u32 %0, %1, %2, %3;" : "=r"(r) : "r"(hi), "r"(m), "r"(l));
    return r;
}

// Tail candidate t of thread (warp, lane): the candidates outside the 2R x 2R register
// tiling — column dx = +R (dy < R) and row dy = +R (dx < R); the corner (R, R) is split
// over warp 0.  Row tails of one warp read consecutive dx (conflict-free words).
template <int R>
__device__ __forceinline__ bool tail_candidate(int warp, int lane, int t, int& dx, int& dy) {
    constexpr int nw = MeGeom<R>::kWarps;
    const bool col = nw == 4 ? warp < 2 : nw == 2 ? warp == 0 : t == 0;
    const int k = nw == 4 ? 32 * (warp & 1) + lane : lane;
    dx = col ? R : -R + k;
    dy = col ? -R + k : R;
    return col;
}

// Tail candidate t of thread (warp, lane) as (column?, k): a column tail has dy = dy0 + k, a
// row tail dx = dx0 + k, in the candidate frame whose main block starts at (dx0, dy0).
template <int R>
__device__ __forceinline__ bool tail_slot(int warp, int lane, int t, int& k) {
    int dx, dy;
    const bool col = tail_candidate<R>(warp, lane, t, dx, dy);
    k = col ? dy + R : dx + R;
    return col;
}

// Border macroblocks (one-warp CTAs, class order only).  When the valid displacements of a
// macroblock fit in R + 1 columns (or rows) — the first / last macroblock column (row) of a
// frame whose width (height) is a multiple of 16 — at most half of the 2R x 2R main candidates
// can be valid: the thread tile then shrinks to TX = 2 dx (TY = 4 dy) candidates over a
// candidate frame starting at dx0 (dy0), so the warp computes the valid half instead of
// computing and masking all of it (CIF +-16: 76 of 396 macroblocks, 9 % of the SAD work).
// Candidates dx = dx0 + p + 4 (TX g + j), dy = dy0 + TY d + i; column tails at dx = dx0 +
// 4 TX kGx, row tails at dy = dy0 + TY kDy; invalid ones never enter the key.  Returns the
// thread's minimal key.  (Out of line: the interior path keeps its registers and code layout.)
#ifndef SP_ME_BINLINE  // A/B knob: the border search inlined measured the same (76.6 %, r5d)
#define SP_ME_BINLINE 0
#endif
template <int R, int TX, int TY>
#if SP_ME_BINLINE
__device__ __forceinline__
#else
__device__ __noinline__
#endif
uint32_t border_search(const uint8_t* smem, int s, int dx0, int dy0, int dxlo, int dxhi,
                                               int dylo, int dyhi, int tid) {
    using G = MeGeom<R>;
    static_assert(G::kWarps == 1, "border search: one-warp CTAs");
    // (the kernel's shared-memory layout: raw window / byte-phase copies / current block)
    auto phase_base = [&](int ph) -> const uint8_t* {
        return ph == 0 ? smem + s * G::kCopy
                       : smem + G::kOffPh + (3 * (G::kPhaseSets == 1 ? 0 : s) + ph - 1) * G::kSlot + 32 * ph;
    };
    const uint4* cq = reinterpret_cast<const uint4*>(smem + G::kOffCur + s * 256);
    constexpr int win = G::kWin;
    constexpr int kDy = G::kThreads / (4 * G::kGx);
    constexpr int NW = TX + 3;
    const int lane = tid & 31, warp = tid >> 5;
    const int p = tid & 3, g = (tid >> 2) % G::kGx, d = tid / (4 * G::kGx);
    const int CX = dx0 + 4 * TX * G::kGx, CY = dy0 + TY * kDy;  // tail column / row
    // tails: window address (row dy + R, byte dx + R of the matching phase copy) and key bits
    const uint8_t* tp[G::kTailPer];
    uint32_t ttie[G::kTailPer];
    bool tval[G::kTailPer];
#pragma unroll
    for (int t = 0; t < G::kTailPer; ++t) {
        int k;
        const bool col = tail_slot<R>(warp, lane, t, k);
        const bool inside = k < (col ? TY * kDy : 4 * TX * G::kGx);  // (beyond: not a candidate)
        const int dx = col ? CX : dx0 + k, dy = col ? dy0 + k : CY;
        tval[t] = inside && dx >= dxlo && dx <= dxhi && dy >= dylo && dy <= dyhi;
        ttie[t] = tie_bits(dx, dy, R);
        tp[t] = inside ? phase_base((dx + R) & 3) + (dy + R) * win + 4 * ((dx + R) >> 2) : phase_base(0);
    }
    uint32_t acc[TX][TY], ta[G::kTailPer];
#pragma unroll
    for (int j = 0; j < TX; ++j)
#pragma unroll
        for (int i = 0; i < TY; ++i) acc[j][i] = 0;
#pragma unroll
    for (int t = 0; t < G::kTailPer; ++t) ta[t] = 0;
    const uint8_t* rowp = phase_base(p) + (dy0 + R + TY * d) * win + 4 * ((dx0 + R) / 4 + TX * g);
    uint32_t Rw[TY][NW];
    auto load_row = [&](uint32_t(&w)[NW], const uint8_t* src) {
        if constexpr (TX == 4) {
            const uint4 a = *reinterpret_cast<const uint4*>(src);
            const uint4 b = *reinterpret_cast<const uint4*>(src + 16);
            w[0] = a.x; w[1] = a.y; w[2] = a.z; w[3] = a.w; w[4] = b.x; w[5] = b.y; w[6] = b.z;
        } else {  // 8-byte aligned: (dx0 + R) and 8 g are multiples of 8
            const uint2 a = *reinterpret_cast<const uint2*>(src);
            const uint2 b = *reinterpret_cast<const uint2*>(src + 8);
            w[0] = a.x; w[1] = a.y; w[2] = b.x; w[3] = b.y; w[4] = *reinterpret_cast<const uint32_t*>(src + 16);
        }
    };
#pragma unroll
    for (int rr = 0; rr < TY - 1; ++rr) load_row(Rw[rr], rowp + rr * win);
#pragma unroll 1
    for (int vb = 0; vb < kMB; vb += TY) {
#pragma unroll
        for (int vv = 0; vv < TY; ++vv) {
            const int v = vb + vv;
            load_row(Rw[(vv + TY - 1) % TY], rowp + (v + TY - 1) * win);
            const uint4 cv = cq[v];
            const uint32_t Cv[4] = {cv.x, cv.y, cv.z, cv.w};
#pragma unroll
            for (int t = 0; t < G::kTailPer; ++t) {
                const uint32_t* tq = reinterpret_cast<const uint32_t*>(tp[t] + v * win);
#pragma unroll
                for (int k = 0; k < 4; ++k) ta[t] = sad4(tq[k], Cv[k], ta[t]);
            }
#pragma unroll
            for (int k = 0; k < 4; ++k)
#pragma unroll
                for (int i = 0; i < TY; ++i)
#pragma unroll
                    for (int j = 0; j < TX; ++j) acc[j][i] = sad4(Rw[(vv + i) % TY][j + k], Cv[k], acc[j][i]);
        }
    }
    uint32_t key = 0xffffffffu;
#pragma unroll
    for (int j = 0; j < TX; ++j) {
        const int dx = dx0 + p + 4 * (TX * g + j);
#pragma unroll
        for (int i = 0; i < TY; ++i) {
            const int dy = dy0 + TY * d + i;
            if (dx >= dxlo && dx <= dxhi && dy >= dylo && dy <= dyhi)
                key = min(key, acc[j][i] * kKeyMul + tie_bits(dx, dy, R));
        }
    }
#pragma unroll
    for (int t = 0; t < G::kTailPer; ++t)
        if (tval[t]) key = min(key, ta[t] * kKeyMul + ttie[t]);
    return key;
}

// Frames still streaming in (sp_me_search_host): wait for a pair's ready flag (relaxed poll,
// then an acquire and a proxy fence order the observed copy before the TMA reads that follow).
// Out of line: the common device-resident path keeps its register / uniform-datapath layout.
__device__ __noinline__ void wait_ready(const int32_t* flag) {
    const long long t0 = clock64();
    while (ld_relaxed_gpu(flag) == 0) {
        __nanosleep(256);
        if (clock64() - t0 > (40ll << 30)) __trap();
    }
    (void)ld_acquire_gpu(flag);  // (flags only go 0 -> 1)
    fence_proxy_async_global();
}

// kMode: kPlain (device-resident frames), kStream (frames still streaming in: ready flags),
// kGather (results all-gathered into every rank's outputs over peer memory).  Separate
// instantiations keep the common path's register and uniform-datapath layout untouched.
enum { kPlain = 0, kStreamed = 1, kGather = 2 };

template <int R, int kMode>
__global__ void __launch_bounds__(MeGeom<R>::kThreads, MeGeom<R>::kMinBlocks)
me_sad_kernel(const __grid_constant__ CUtensorMap ref_map, const __grid_constant__ CUtensorMap cur_map, MeArgs A,
              const __grid_constant__ GatherArgs X) {
    using G = MeGeom<R>;
    constexpr int kTy = G::kTy;  // (shadows the R = 32 default)
    constexpr bool kStream = kMode == kStreamed;
    constexpr int win = G::kWin;
    constexpr int side = 2 * R + 1;
    constexpr int nwarps = G::kWarps;
    extern __shared__ __align__(128) uint8_t smem_raw[];
    __shared__ __align__(8) uint64_t full[2];
    __shared__ uint32_t red32[2][nwarps];  // per-stage per-warp minimal key
    __shared__ uint32_t lsum[2];           // per-stage SAD of the corner candidate (R, R)
    __shared__ uint32_t ltie[2];           // (one-warp CTAs) its tie bits, ~0u if invalid
    // align to 128 bytes by offsetting the shared pointer itself (keeps LDS/STS addressing)
    uint8_t* smem = smem_raw + ((128u - (smem_addr(smem_raw) & 127u)) & 127u);

    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const uint32_t mbx = (uint32_t)A.mbx;
    const uint32_t per_pair = (uint32_t)A.mb_rows * mbx;
    const uint32_t total = A.total_mb;  // host guarantees < 2^31
    const uint32_t Gs = gridDim.x;
    const int W = A.width, Hf = A.frame_height;
    // byte phase ph of stage st (ph = 0: the TMA'd window).  Copy ph starts 32*ph bytes past
    // a 128-byte boundary, so the four phases a quarter warp reads hit distinct banks.
    auto phase_copy = [&](int st, int ph) -> uint8_t* {
        return ph == 0 ? smem + st * G::kCopy
                       : smem + G::kOffPh + (3 * (G::kPhaseSets == 1 ? 0 : st) + ph - 1) * G::kSlot + 32 * ph;
    };
    struct Pos {
        int pair, byr, bx;
    };
    auto locate = [&](uint32_t mb) -> Pos {
#if SP_ME_SCRAMBLE
        // column-major over the launch's macroblock rows: consecutive grabs come from
        // different rows, so the border rows (whose dead warps skip their main candidates)
        // spread over the whole launch instead of coinciding on every SM
        const uint32_t col = mb / A.nrows, f = mb - col * A.nrows + A.flat_mb0 / mbx;
        const uint32_t pair = f / (uint32_t)A.mb_rows;
        return Pos{(int)pair, (int)(f - pair * (uint32_t)A.mb_rows), (int)col};
#else
        if constexpr (nwarps == 1) {
            if (A.border_order) {  // class order (MeArgs::border_order; whole frames, flat_mb0 = 0)
                const uint32_t mbx2 = mbx - 2, rows2 = (uint32_t)A.mb_rows - 2;
                if (mb < A.cls_end[0]) {  // interior
                    const uint32_t pair = fdiv(mb, A.div_int), k = mb - pair * (rows2 * mbx2);
                    const uint32_t r = fdiv(k, A.div_icols);
                    return Pos{(int)pair, (int)(1 + r), (int)(1 + k - r * mbx2)};
                }
                if (mb < A.cls_end[1]) {  // top / bottom rows without the corners
                    const uint32_t m = mb - A.cls_end[0], pair = fdiv(m, A.div_rows2), k = m - pair * 2 * mbx2;
                    const bool top = k < mbx2;
                    return Pos{(int)pair, top ? 0 : (int)rows2 + 1, (int)(1 + (top ? k : k - mbx2))};
                }
                if (mb < A.cls_end[2]) {  // left / right columns without the corners
                    const uint32_t m = mb - A.cls_end[1], pair = fdiv(m, A.div_cols2), k = m - pair * 2 * rows2;
                    const bool left = k < rows2;
                    return Pos{(int)pair, (int)(1 + (left ? k : k - rows2)), left ? 0 : (int)mbx - 1};
                }
                const uint32_t m = mb - A.cls_end[2];  // corners
                return Pos{(int)(m >> 2), (m & 2) ? (int)rows2 + 1 : 0, (m & 1) ? (int)mbx - 1 : 0};
            }
        }
        mb += A.flat_mb0;
        const uint32_t pair = fdiv(mb, A.div_per_pair), rem = mb - pair * per_pair;
        const uint32_t byr = fdiv(rem, A.div_mbx);
        return Pos{(int)pair, (int)byr, (int)(rem - byr * mbx)};
#endif
    };
    // (kStream, thread 0) highest pair seen ready: the copies land in frame order and a CTA's
    // macroblocks come in increasing pair order, so each pair's flag is polled (and fenced)
    // once per CTA instead of once per macroblock
    int ready_seen = -1;
    auto issue = [&](uint32_t mb, int st) {  // single thread: stage the window + cur of mb
        const Pos q = locate(mb);
        if (kStream && q.pair > ready_seen) {
            wait_ready(A.ready + q.pair);
            ready_seen = q.pair;
        }
        const int x0 = kMB * q.bx, y0 = kMB * (A.mb_row_begin + q.byr);
        mbar_arrive_expect_tx(&full[st], (uint32_t)(G::kCopy + kMB * kMB));
        tma_load_3d(smem + st * G::kCopy, &ref_map, x0 - R + A.pad, y0 - R - A.row0 + A.pad, q.pair - A.pair_base,
                    &full[st]);
        tma_load_3d(smem + G::kOffCur + st * 256, &cur_map, x0 + A.pad, y0 - A.row0 + A.pad, q.pair - A.pair_base,
                    &full[st]);
    };
    bool gather_armed = false;  // (kGather, finalizing thread) every rank's ready flag seen for this epoch
    // publish macroblock mbp's argmin from stage sp (every warp's key + the corner candidate)
    auto finalize = [&](uint32_t mbp, int sp) {
        uint32_t b = red32[sp][0];
#pragma unroll
        for (int w = 1; w < nwarps; ++w) b = min(b, red32[sp][w]);
        const uint32_t lsad = lsum[sp];
        const Pos q = locate(mbp);
        bool lvalid;
        if constexpr (nwarps == 1) {  // the corner candidate of the searched frame (border search: moved)
            const uint32_t lt = ltie[sp];
            lvalid = lt != 0xffffffffu;
            if (lvalid) b = min(b, lsad * kKeyMul + lt);
        } else {
            const int x0 = kMB * q.bx, y0 = kMB * (A.mb_row_begin + q.byr);
            lvalid = A.unrestricted || ((x0 + R + 16 <= W) && (y0 + R + 16 <= Hf));
            if (lvalid) b = min(b, lsad * kKeyMul + tie_bits(R, R, R));
        }
        const size_t idx = ((size_t)q.pair * A.mb_rows + q.byr) * mbx + q.bx;
        const uint32_t sad = b / kKeyMul, tie = b - sad * kKeyMul;
        const int dy = (int)((tie >> 1) & 127) - R;
        const int adx = (int)((tie >> 8) & 127) - abs(dy);
        // (dx, dy) as one 32-bit store (the outputs may be mapped host memory: fewer PCIe writes)
        const uint32_t mvw = (uint32_t)(uint16_t)((tie & 1) ? adx : -adx) | ((uint32_t)(uint16_t)dy << 16);
        *reinterpret_cast<uint32_t*>(A.mv + 2 * idx) = mvw;
        A.sad[idx] = sad;
        if constexpr (kMode == kGather) {
            // all-gather: the same 8 bytes into every other rank's outputs (peer stores), once
            // those ranks have announced (ready) that their outputs of the previous epoch are free
            if (!gather_armed) {
                const long long t0 = clock64();
                for (int q = 0; q < X.nranks; ++q)
                    while (ld_acquire_sys(X.flags[X.rank] + q) < X.epoch) {
                        __nanosleep(128);
                        if (clock64() - t0 > (40ll << 30)) __trap();
                    }
                gather_armed = true;
            }
            for (int q = 0; q < X.nranks; ++q) {
                if (q == X.rank) continue;
                *reinterpret_cast<uint32_t*>(X.mv[q] + 2 * idx) = mvw;
                X.sad[q][idx] = sad;
            }
        }
        if (A.surface) A.surface[idx * side * side + (size_t)side * side - 1] = lvalid ? lsad : 0xffffffffu;
    };

#if SP_ME_EXP & 32
    if (tid == 0 && blockIdx.x < 4096) {
        unsigned sm;
        asm volatile("mov.u32 %0, %%smid;" : "=r"(sm));
        g_me_cta[blockIdx.x][0] = sm;
        g_me_cta[blockIdx.x][1] = globaltimer();
    }
#endif
    if (kMode == kGather && blockIdx.x == 0 && tid == 0) {
        // this rank's outputs of the previous epoch are no longer read (stream order): let
        // every rank write this epoch's results into them
        for (int q = 0; q < X.nranks; ++q) st_release_sys(X.flags[q] + X.rank, X.epoch);
    }
    if (tid == 0) {
        prefetch_tmap(&ref_map);
        prefetch_tmap(&cur_map);
        mbar_init(&full[0], 1);
        mbar_init(&full[1], 1);
        fence_mbar_init();
        if (blockIdx.x < total) issue(blockIdx.x, 0);
    }
    __syncthreads();

    // thread's candidate tile: dx = -R + p + 4*(4g + j), dy = -R + 8d + i (a quarter warp
    // spans the four byte phases: conflict-free LDS.128)
    const int p = tid & 3, g = (tid >> 2) % G::kGx, d = tid / (4 * G::kGx);
    // per-thread constants of the epilogue, kept in shared memory instead of registers:
    // tie bits A_j = |dx_j| << 8 | (dx_j > 0) per (p, g), B_i = |dy_i| << 8 | (dy_i + R) << 1
    // per d (tie(j, i) = A_j + B_i, no carries between the fields)
    constexpr int kDy = G::kThreads / (4 * G::kGx);
    __shared__ uint4 tieA[4 * G::kGx];
    __shared__ uint4 tieB[kDy][kTy / 4];
    if (tid < 4 * G::kGx) {
        uint32_t a[4];
        for (int j = 0; j < 4; ++j) {
            const int dx = -R + (tid & 3) + 4 * (4 * (tid >> 2) + j);
            a[j] = ((uint32_t)abs(dx) << 8) | (dx > 0 ? 1u : 0u);
        }
        tieA[tid] = make_uint4(a[0], a[1], a[2], a[3]);
    }
    if (tid < kDy) {
        uint32_t b[kTy];
        for (int i = 0; i < kTy; ++i) {
            const int dy = -R + kTy * tid + i;
            b[i] = ((uint32_t)abs(dy) << 8) | ((uint32_t)(dy + R) << 1);
        }
        for (int q = 0; q < kTy / 4; ++q) tieB[tid][q] = make_uint4(b[4 * q], b[4 * q + 1], b[4 * q + 2], b[4 * q + 3]);
    }
    // tail candidates: tie bits and staged-copy offsets (stage 0, stage 1), per thread.  Two
    // offsets even with one phase-copy set: a tail of byte phase 0 reads the TMA'd window
    // itself, which alternates between the two stages (one-warp CTAs read stage 0's window on
    // every macroblock until round-2 session 3 — wrong tails from a CTA's second macroblock on).
    // One-warp CTAs pack the two 16-bit offsets into one word (shared memory holds them at 16
    // CTAs per SM: 14,464 of the 14,592 bytes each may take)
    constexpr bool kPackT = G::kPhaseSets == 1;
    __shared__ uint32_t tinfo[G::kTailPer][kPackT ? 2 : 3][G::kThreads];
#pragma unroll
    for (int t = 0; t < G::kTailPer; ++t) {
        int dxt, dyt;
        tail_candidate<R>(warp, lane, t, dxt, dyt);
        tinfo[t][0][tid] = tie_bits(dxt, dyt, R);
#pragma unroll
        for (int st = 0; st < 2; ++st) {
            const uint32_t off =
                (uint32_t)(phase_copy(st, (dxt + R) & 3) - smem) + (dyt + R) * win + 4 * ((dxt + R) >> 2);
            if (!kPackT) tinfo[t][1 + st][tid] = off;
            else if (st == 0) tinfo[t][1][tid] = off;
            else tinfo[t][1][tid] |= off << 16;
        }
    }
    // macroblock index and position (pair, MB row, MB column) per stage, written by thread 0
    // one macroblock ahead (before the barrier that precedes their reading)
    __shared__ Pos posS[2];
    __shared__ uint32_t mbS[2];
    if (tid == 0) {
        posS[0] = locate(blockIdx.x < total ? blockIdx.x : 0);
        mbS[0] = blockIdx.x;
    }
    __syncthreads();
#if SP_ME_EXP & 16
    __shared__ unsigned prof_s[nwarps][8];
    if (lane == 0)
        for (int k = 0; k < 8; ++k) prof_s[warp][k] = 0;
    unsigned t_prev = (unsigned)clock();
#endif
    int it = 0;
    uint32_t prev_mb = 0;
    for (uint32_t mb = blockIdx.x; mb < total; ++it) {
        const int s = it & 1;
        // the next macroblock of this CTA, published in mbS[s^1] before this iteration's barrier
        // (the atomic's latency hides under the move-in wait and the phase build)
        if (tid == 0) mbS[s ^ 1] = atomicAdd(A.counter, 1u) + Gs;
        mbar_wait(&full[s], (it >> 1) & 1);
        if (G::kPhaseSets == 1) __syncwarp();  // every lane done reading the single phase set
        PMARK(0);
        if (!(SP_ME_EXP & 128)) {  // (128: timing-only build without the phase build)
            // byte-phase copies (word q of copy p = bytes [4q+p, 4q+p+4) of the row):
            // (row, phase) units spread over the CTA, one window row loaded per unit
            constexpr int v4_per_row = win / 16;
            const uint8_t* raw = smem + s * G::kCopy;
#pragma unroll
            for (int k = 0; k < (3 * win + G::kThreads - 1) / G::kThreads; ++k) {
                const int u = tid + k * G::kThreads;
                if (u < 3 * win) {
                    const int ph = 1 + u / win, r = u - (ph - 1) * win;
                    const uint4* rowv = reinterpret_cast<const uint4*>(raw + r * win);
                    uint4 wv[v4_per_row];
#pragma unroll
                    for (int c = 0; c < v4_per_row; ++c) wv[c] = rowv[c];
                    uint4* out = reinterpret_cast<uint4*>(phase_copy(s, ph) + r * win);
#if SP_ME_PHASE_FMA
                    const uint32_t m = 1u << (32 - 8 * ph);
#endif
#pragma unroll
                    for (int c = 0; c < v4_per_row; ++c) {
                        const uint32_t nx = c + 1 < v4_per_row ? wv[c + 1].x : 0u;
                        uint4 o;
#if SP_ME_PHASE_FMA
                        o.x = shr_bytes_fma(wv[c].x, wv[c].y, m);
                        o.y = shr_bytes_fma(wv[c].y, wv[c].z, m);
                        o.z = shr_bytes_fma(wv[c].z, wv[c].w, m);
                        o.w = shr_bytes_fma(wv[c].w, nx, m);
#else
                        o.x = __funnelshift_r(wv[c].x, wv[c].y, 8 * ph);
                        o.y = __funnelshift_r(wv[c].y, wv[c].z, 8 * ph);
                        o.z = __funnelshift_r(wv[c].z, wv[c].w, 8 * ph);
                        o.w = __funnelshift_r(wv[c].w, nx, 8 * ph);
#endif
                        out[c] = o;
                    }
                }
            }
        }
        PMARK(1);
        // the only CTA barrier per macroblock: phase copies of stage s complete; every warp
        // is done with stage s^1 (previous macroblock) and has posted its key for it
        __syncthreads();
        const uint32_t next_mb = mbS[s ^ 1];
        if (tid == 0 && next_mb < total) {
            fence_proxy_async_smem();
            issue(next_mb, s ^ 1);
            posS[s ^ 1] = locate(next_mb);
        }
        if (tid == G::kThreads - 32 && it > 0) finalize(prev_mb, s ^ 1);
        PMARK(2);

#if SP_ME_EXP & 64  // race stress (tests/test_me_stress_gpu.py): the upper warps start late, so the
        // lower ones build the next macroblock's copies while these still read this one's
        if (warp >= nwarps / 2) __nanosleep(20000);
#endif
        // ---- validity (restricted vectors) only matters near the frame border ----------
        const Pos q = posS[s];  // (written one macroblock ahead; stable until the next barrier)
        const int x0 = kMB * q.bx, y0 = kMB * (A.mb_row_begin + q.byr);
        const int dxlo = -x0 > -R ? -x0 : -R, dxhi = W - 16 - x0 < R ? W - 16 - x0 : R;
        const int dylo = -y0 > -R ? -y0 : -R, dyhi = Hf - 16 - y0 < R ? Hf - 16 - y0 : R;
        const bool interior = A.unrestricted || (dxlo == -R && dxhi == R && dylo == -R && dyhi == R);
        // a warp whose whole band of main dy candidates is invalid skips them (warp-uniform;
        // 4-warp CTAs: warp w holds dy in [-R + 16 w, -R + 16 w + 15]); its tails still run
        bool main_dead = false;
        if (SP_ME_SKIP && nwarps > 1 && !interior && !A.surface) {
            constexpr int kDyWarp = (32 / (4 * G::kGx)) * kTy;  // dy values of a warp's main candidates
            const int blo = -R + kDyWarp * warp, bhi = blo + kDyWarp - 1;
            main_dead = bhi < dylo || blo > dyhi;
        }
        // the corner candidate of the searched frame — (R, R), or the moved corner of a border
        // search: 64 (row, word) pieces over warp 0 (one-warp CTAs also post its tie bits)
        auto corner = [&](int cx, int cy, bool cvalid) {
            const uint32_t* rw = reinterpret_cast<const uint32_t*>(smem + s * G::kCopy + (cy + R) * win) + (cx + R) / 4;
            const uint4* cq4 = reinterpret_cast<const uint4*>(smem + G::kOffCur + s * 256);
            uint32_t part = 0;
#pragma unroll
            for (int o = lane; o < 64; o += 32) {
                const int v = o >> 2, k = o & 3;
                const uint4 cv = cq4[v];
                const uint32_t cw = k == 0 ? cv.x : k == 1 ? cv.y : k == 2 ? cv.z : cv.w;
                part = sad4(rw[v * (win / 4) + k], cw, part);
            }
            const uint32_t tot = __reduce_add_sync(0xffffffffu, part);
            if (lane == 0) {
                lsum[s] = tot;
                if constexpr (nwarps == 1) ltie[s] = cvalid ? tie_bits(cx, cy, R) : 0xffffffffu;
            }
        };
        uint32_t key = 0xffffffffu;
        bool bsearch = false;  // (class order, one-warp CTAs) this macroblock took a half-frame border search
        if constexpr (nwarps == 1) {
            if (A.border_order && !interior) {
                // valid dx within R + 1 columns from an 8-byte-aligned origin, or dy within R + 1 rows
                const int cx = dxlo - ((dxlo + R) & 7);
                const bool hx = dxhi <= cx + R, hy = dyhi - dylo <= R;
                if (hx || hy) {
                    const int dx0 = hx ? cx : -R, dy0 = hy ? dylo : -R;
                    const int CX = dx0 + (hx ? R : 2 * R), CY = dy0 + (hy ? R : 2 * R);
                    if (hx && hy) key = border_search<R, 2, 4>(smem, s, dx0, dy0, dxlo, dxhi, dylo, dyhi, tid);
                    else if (hx) key = border_search<R, 2, 8>(smem, s, dx0, dy0, dxlo, dxhi, dylo, dyhi, tid);
                    else key = border_search<R, 4, 4>(smem, s, dx0, dy0, dxlo, dxhi, dylo, dyhi, tid);
                    corner(CX, CY, CX >= dxlo && CX <= dxhi && CY >= dylo && CY <= dyhi);
                    bsearch = true;
                }
            }
        }
        if (!bsearch) {
        // ---- 2R x 2R main candidates (4 dx of one byte phase x 8 dy per thread) plus this
        //      thread's tail candidates, all in one row loop ----
        uint32_t acc[kTx][kTy];
#pragma unroll
        for (int j = 0; j < kTx; ++j)
#pragma unroll
            for (int i = 0; i < kTy; ++i) acc[j][i] = 0;
        uint32_t ta[G::kTailPer];
        const uint8_t* tp[G::kTailPer];
#pragma unroll
        for (int t = 0; t < G::kTailPer; ++t) {
            tp[t] = smem + (kPackT ? (tinfo[t][1][tid] >> (16 * s)) & 0xffffu : tinfo[t][1 + s][tid]);
            ta[t] = 0;
        }
        if (main_dead) {  // tails only (one LDS.128 of the current row, 4 LDS.32 + 4 SADs per tail)
            const uint4* cq = reinterpret_cast<const uint4*>(smem + G::kOffCur + s * 256);
#pragma unroll 4
            for (int v = 0; v < kMB; ++v) {
                const uint4 cv = cq[v];
                const uint32_t Cv[4] = {cv.x, cv.y, cv.z, cv.w};
#pragma unroll
                for (int t = 0; t < G::kTailPer; ++t) {
                    const uint32_t* tq = reinterpret_cast<const uint32_t*>(tp[t] + v * win);
#pragma unroll
                    for (int k = 0; k < 4; ++k) ta[t] = sad4(tq[k], Cv[k], ta[t]);
                }
            }
        } else {
            // Candidate (j, i) compares cur row v with window row 8d + i + v.  Loop over v with
            // a ring of the 8 window rows in use (row rho in slot rho & 7, 7 words each: the
            // 4 dx candidates x 4 words of one byte phase); body unrolled 8x so every ring
            // index is static, outer loop rolled to halve the code (I-cache).  Innermost
            // order (k, i, j) makes consecutive VABSDIFF4s independent.
            const uint8_t* rowp = phase_copy(s, p) + (kTy * d) * win + 16 * g;
            const uint4* cq = reinterpret_cast<const uint4*>(smem + G::kOffCur + s * 256);
            uint32_t Rw[kTy][7];  // words 4g..4g+6 (j + k <= 6)
#pragma unroll
            for (int rr = 0; rr < kTy - 1; ++rr) {
                const uint4 w0 = *reinterpret_cast<const uint4*>(rowp + rr * win);
                const uint4 w1 = *reinterpret_cast<const uint4*>(rowp + rr * win + 16);
                Rw[rr][0] = w0.x; Rw[rr][1] = w0.y; Rw[rr][2] = w0.z; Rw[rr][3] = w0.w;
                Rw[rr][4] = w1.x; Rw[rr][5] = w1.y; Rw[rr][6] = w1.z;
            }
#pragma unroll 1
            for (int vb = 0; vb < ((SP_ME_EXP & 8) ? 4 * kMB : kMB); vb += kTy) {
#pragma unroll
                for (int vv = 0; vv < kTy; ++vv) {
                    const int v = ((SP_ME_EXP & 8) ? (vb & (kMB - 1)) : vb) + vv;
                    {
                        const int slot = (vv + kTy - 1) % kTy;
                        const uint4 w0 = *reinterpret_cast<const uint4*>(rowp + (v + kTy - 1) * win);
                        const uint4 w1 = *reinterpret_cast<const uint4*>(rowp + (v + kTy - 1) * win + 16);
                        Rw[slot][0] = w0.x; Rw[slot][1] = w0.y; Rw[slot][2] = w0.z; Rw[slot][3] = w0.w;
                        Rw[slot][4] = w1.x; Rw[slot][5] = w1.y; Rw[slot][6] = w1.z;
                    }
                    const uint4 cv = cq[v];
                    const uint32_t Cv[4] = {cv.x, cv.y, cv.z, cv.w};
                    if (!(SP_ME_EXP & 2)) {
#pragma unroll
                        for (int t = 0; t < G::kTailPer; ++t) {
                            // four LDS.32 for every tail (one uniform path: a predicated
                            // LDS.128 variant for the aligned column costs more issue slots
                            // than the column's 4-way bank conflicts)
                            const uint32_t* tq = reinterpret_cast<const uint32_t*>(tp[t] + v * win);
                            const uint32_t tw[4] = {tq[0], tq[1], tq[2], tq[3]};
#pragma unroll
                            for (int k = 0; k < 4; ++k) ta[t] = sad4(tw[k], Cv[k], ta[t]);
                        }
                    }
#pragma unroll
                    for (int k = 0; k < 4; ++k)
#pragma unroll
                        for (int i = 0; i < kTy; ++i)
#pragma unroll
                            for (int j = 0; j < kTx; ++j)
                                acc[j][i] = sad4(Rw[(vv + i) % kTy][j + k], Cv[k], acc[j][i]);
                }
            }
        }
        PMARK(3);
        if (warp == 0) corner(R, R, A.unrestricted || (dxhi >= R && dyhi >= R));
        PMARK(4);
        if (!interior) {
#pragma unroll
            for (int j = 0; j < kTx; ++j) {
                const int dx = -R + p + 4 * (4 * g + j);
#pragma unroll
                for (int i = 0; i < kTy; ++i) {
                    const int dy = -R + kTy * d + i;
                    if (dx < dxlo || dx > dxhi || dy < dylo || dy > dyhi) acc[j][i] = kInvalidSad;
                }
            }
#pragma unroll
            for (int t = 0; t < G::kTailPer; ++t) {
                int dx, dy;
                tail_candidate<R>(warp, lane, t, dx, dy);
                if (dx < dxlo || dx > dxhi || dy < dylo || dy > dyhi) ta[t] = kInvalidSad;
            }
        }
        if (A.surface) {
            uint32_t* sf = A.surface + (((size_t)q.pair * A.mb_rows + q.byr) * mbx + q.bx) * side * side;
#pragma unroll
            for (int j = 0; j < kTx; ++j)
#pragma unroll
                for (int i = 0; i < kTy; ++i)
                    sf[(kTy * d + i) * side + (p + 4 * (4 * g + j))] = acc[j][i] == kInvalidSad ? 0xffffffffu : acc[j][i];
#pragma unroll
            for (int t = 0; t < G::kTailPer; ++t) {
                int dx, dy;
                tail_candidate<R>(warp, lane, t, dx, dy);
                sf[(dy + R) * side + (dx + R)] = ta[t] == kInvalidSad ? 0xffffffffu : ta[t];
            }
        }
        // ---- argmin: min over this thread's keys, key(j, i) = acc * kKeyMul + A_j + B_i,
        //      then one CREDUX per warp ----
        {
            const uint4 a4 = tieA[p + 4 * g];
            const uint32_t Aj[4] = {a4.x, a4.y, a4.z, a4.w};
            uint32_t Bi[kTy];
#pragma unroll
            for (int q = 0; q < kTy / 4; ++q) {
                const uint4 bq = tieB[d][q];
                Bi[4 * q] = bq.x;
                Bi[4 * q + 1] = bq.y;
                Bi[4 * q + 2] = bq.z;
                Bi[4 * q + 3] = bq.w;
            }
#pragma unroll
            for (int i = 0; i < kTy; ++i) {
                uint32_t ki = 0xffffffffu;
#pragma unroll
                for (int j = 0; j < kTx; ++j) ki = min(ki, acc[j][i] * kKeyMul + Aj[j]);
                key = min(key, ki + Bi[i]);
            }
        }
#pragma unroll
        for (int t = 0; t < G::kTailPer; ++t) key = min(key, ta[t] * kKeyMul + tinfo[t][0][tid]);
        }  // (full-frame search)
        key = __reduce_min_sync(0xffffffffu, key);
        if (lane == 0) red32[s][warp] = key;
        PMARK(7);
        prev_mb = mb;
        mb = next_mb;
    }
#if SP_ME_EXP & 16
    if (lane == 0)
        for (int k = 0; k < 8; ++k) atomicAdd(&g_me_prof[k], (unsigned long long)prof_s[warp][k]);
#endif
    __syncthreads();
    if (tid == G::kThreads - 32 && it > 0) finalize(prev_mb, (it - 1) & 1);
    if (kMode == kGather) __syncthreads();  // the last finalize's peer stores precede the fence below
    if (tid == 0) {
        // self-resetting counter: every grab of this CTA precedes its arrival here, so the
        // last CTA to arrive sees all of them done and zeroes both words for the next launch
        // on this stream (no per-launch memset)
        if (kMode == kGather) __threadfence_system();
        else __threadfence();
        if (atomicAdd(A.counter + 1, 1u) == Gs - 1) {
            if (kMode == kGather) {
                // every CTA's results are out (each fenced before its arrival): tell every rank
                __threadfence_system();
                for (int q = 0; q < X.nranks; ++q) st_release_sys(X.flags[q] + X.nranks + X.rank, X.epoch);
            } else {
                __threadfence();
            }
            A.counter[0] = 0;
            A.counter[1] = 0;
        }
    }
#if SP_ME_EXP & 32
    if (tid == 0 && blockIdx.x < 4096) g_me_cta[blockIdx.x][2] = globaltimer();
#endif
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
        const int gy = y0 - R + wy - A.row0 + A.pad, gx = x0 - R + wx + A.pad;
        uint8_t v = 0;
        if (gy >= 0 && gy < rows_in_buffer && gx >= 0 && gx < A.width + 2 * A.pad) v = rp[(int64_t)gy * pitch + gx];
        win_s[q] = v;
    }
    for (int q = tid; q < kMB * kMB; q += nthr)
        cur_s[q] = cp[(int64_t)(y0 - A.row0 + A.pad + q / kMB) * pitch + x0 + A.pad + q % kMB];
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
        const bool valid = A.unrestricted ||
                           ((x0 + dx >= 0) && (x0 + dx + 16 <= A.width) && (y0 + dy >= 0) && (y0 + dy + 16 <= A.frame_height));
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

// The fast kernel's macroblock counter: two words (grab counter, CTAs finished) per
// (device, stream), library-owned, zero between launches (the kernel resets them: see the end
// of me_sad_kernel), so launches on one stream reuse their slot and launches on different
// streams never share one.  A stream handle is assumed not to be destroyed and recreated
// while a launch on it is still running.
constexpr int kMaxDev = 64;
int counter_slot(cudaStream_t s, uint32_t** out) {
    constexpr int kSlots = 4096;
    static std::mutex mu;
    static uint32_t* pool[kMaxDev] = {};
    static std::unordered_map<cudaStream_t, uint32_t*>* slots[kMaxDev] = {};
    int dev = 0;
    SP_CUDA_TRY(cudaGetDevice(&dev));
    if (dev < 0 || dev >= kMaxDev) return SP_ERR_UNSUPPORTED;
    std::lock_guard<std::mutex> lk(mu);
    if (!pool[dev]) {
        void* p = nullptr;
        SP_CUDA_TRY(cudaMalloc(&p, 2 * kSlots * sizeof(uint32_t)));
        SP_CUDA_TRY(cudaMemset(p, 0, 2 * kSlots * sizeof(uint32_t)));
        pool[dev] = static_cast<uint32_t*>(p);
        slots[dev] = new std::unordered_map<cudaStream_t, uint32_t*>();
    }
    auto it = slots[dev]->find(s);
    if (it == slots[dev]->end()) {
        if (slots[dev]->size() >= (size_t)kSlots) return SP_ERR_CAPACITY;  // > 4096 distinct streams
        it = slots[dev]->emplace(s, pool[dev] + 2 * slots[dev]->size()).first;
    }
    *out = it->second;
    return SP_OK;
}

// Per-device launch state of one fast-kernel instantiation: grid cap (occupancy x SMs) and
// the shared-memory attribute, set once per device (the attribute is per device context).
template <int R, int kMode>
int fast_grid_cap(int* cap) {
    using G = MeGeom<R>;
    static std::mutex mu;
    static int caps[kMaxDev] = {};
    int dev = 0;
    SP_CUDA_TRY(cudaGetDevice(&dev));
    if (dev < 0 || dev >= kMaxDev) return SP_ERR_UNSUPPORTED;
    std::lock_guard<std::mutex> lk(mu);
    if (!caps[dev]) {
        int sms = 0, occ = 0;
        SP_CUDA_TRY(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev));
        SP_CUDA_TRY(cudaFuncSetAttribute(me_sad_kernel<R, kMode>, cudaFuncAttributeMaxDynamicSharedMemorySize, G::kSmem));
        SP_CUDA_TRY(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, me_sad_kernel<R, kMode>, G::kThreads, G::kSmem));
        int c = sms * (occ > 0 ? occ : 1);
        // SP_ME_GRID_CAP (sanitizer runs): a few CTAs then walk many macroblocks each, so
        // racecheck sees both pipeline stages in use within one CTA
        if (const char* e = std::getenv("SP_ME_GRID_CAP"))
            if (std::atoi(e) > 0 && std::atoi(e) < c) c = std::atoi(e);
        caps[dev] = c;
    }
    *cap = caps[dev];
    return SP_OK;
}

template <int R, int kMode>
int launch_fast(const CUtensorMap& rm, const CUtensorMap& cm, const MeArgs& a, const GatherArgs& x, int64_t total,
                cudaStream_t s) {
    using G = MeGeom<R>;
    int grid_cap = 0;
    int st = fast_grid_cap<R, kMode>(&grid_cap);
    if (st) return st;
    const int grid = (int)(total < grid_cap ? total : grid_cap);
    me_sad_kernel<R, kMode><<<grid, G::kThreads, G::kSmem, s>>>(rm, cm, a, x);
    return SP_OK;
}

// Encoded tensor maps, cached per (device, base, geometry): encoding is pure host work (a few
// us per map); the map holds only the address and the geometry, so a freed-and-reused address
// with the same geometry yields the same map — no stale entries are possible.
struct MapKey {
    int dev;
    const void* base;
    int64_t w, rows, pairs, pitch, stride, bw, bh;
    bool operator==(const MapKey& o) const {
        return dev == o.dev && base == o.base && w == o.w && rows == o.rows && pairs == o.pairs && pitch == o.pitch &&
               stride == o.stride && bw == o.bw && bh == o.bh;
    }
};
int cached_map(CUtensorMap* m, const uint8_t* base, int32_t width, int32_t rows, int32_t n_pairs, int64_t pitch,
               int64_t pair_stride, uint32_t box_w, uint32_t box_h) {
    constexpr int kEntries = 32;
    static std::mutex mu;
    static MapKey keys[kEntries];
    static CUtensorMap maps[kEntries];
    static int used = 0, next = 0;
    int dev = 0;
    SP_CUDA_TRY(cudaGetDevice(&dev));
    const MapKey k{dev, base, width, rows, n_pairs, pitch, pair_stride, box_w, box_h};
    {
        std::lock_guard<std::mutex> lk(mu);
        for (int i = 0; i < used; ++i)
            if (keys[i] == k) {
                *m = maps[i];
                return SP_OK;
            }
    }
    int st = make_map(m, base, width, rows, n_pairs, pitch, pair_stride, box_w, box_h);
    if (st) return st;
    std::lock_guard<std::mutex> lk(mu);
    keys[next] = k;
    maps[next] = *m;
    next = (next + 1) % kEntries;
    if (used < kEntries) ++used;
    return SP_OK;
}

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

namespace {
int me_search_impl(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width, int32_t rows_in_buffer,
                   int32_t row0_global, int32_t frame_height, int32_t n_pairs, int64_t pair_stride, int32_t block,
                   int32_t range, int32_t mb_row_begin, int32_t mb_row_end, int16_t* mv, uint32_t* best_sad,
                   uint32_t* surface, void* stream, int32_t pad, const int32_t* ready = nullptr) {
    if (block != kMB) return SP_ERR_UNSUPPORTED;
    if (ready && !fast_range(range)) return SP_ERR_UNSUPPORTED;  // streamed frames: fast path only
    if (!ref || !cur || !mv || !best_sad || (reinterpret_cast<uintptr_t>(mv) & 3) ||
        (reinterpret_cast<uintptr_t>(best_sad) & 3))
        return SP_ERR_INVALID_ARG;
    if (range < 0 || range > 63 || width < kMB || frame_height < kMB || n_pairs < 0 || rows_in_buffer < 1)
        return SP_ERR_INVALID_ARG;
    if (pitch < width + 2 * pad || (pitch & 15) || (pair_stride & 15) || (reinterpret_cast<uintptr_t>(ref) & 15) ||
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
    MeArgs a{width, frame_height, row0_global, range, n_pairs, mbx, mb_row_begin, rows, 2 * range + 16, pad,
             pad > 0 ? 1 : 0, mv, best_sad, surface, ready, nullptr, 0u, 0, 0u, 0u};
    const GatherArgs nox{};
    if (fast_range(range)) {
        int st0;
        if ((st0 = counter_slot(s, &a.counter))) return st0;
        CUtensorMap rm, cm;
        int st;
        const int64_t ps = n_pairs > 1 ? pair_stride : pitch * rows_in_buffer;
        if ((st = cached_map(&rm, ref, width + 2 * pad, rows_in_buffer, n_pairs, pitch, ps, (uint32_t)a.win,
                             (uint32_t)a.win)))
            return st;
        if ((st = cached_map(&cm, cur, width + 2 * pad, rows_in_buffer, n_pairs, pitch, ps, kMB, kMB))) return st;
        a.n_pairs = n_pairs;
        const int64_t total = (int64_t)mbx * rows * n_pairs;
        if (total >= (int64_t(1) << 31)) return SP_ERR_UNSUPPORTED;  // 32-bit macroblock indices in the kernel
        a.total_mb = (uint32_t)total;
        a.nrows = (uint32_t)(rows * n_pairs);
        a.div_per_pair = make_fastdiv((uint32_t)(rows * mbx));
        a.div_mbx = make_fastdiv((uint32_t)mbx);
        // class order with half-frame border searches (MeArgs::border_order): R = 16, whole
        // restricted frames on the device, no surface, and enough macroblocks that the class
        // phases are long against one macroblock per CTA (a single CIF pair, M2, keeps the
        // plain order: one wave, where the border macroblocks are not on the critical path).
        // $SP_ME_BORDER = 0 / 1 forces it off / on (whenever eligible) for tests and A/B runs.
        if (range == 16 && !ready && !surface && pad == 0 && mb_row_begin == 0 && rows == mby && mbx >= 3 &&
            mby >= 3) {
            const char* e = std::getenv("SP_ME_BORDER");
            const bool on = e && *e ? std::atoi(e) != 0 : total >= 8192;
            if (on) {
                const uint32_t P = (uint32_t)n_pairs, nI = (uint32_t)((mby - 2) * (mbx - 2));
                a.border_order = 1;
                a.cls_end[0] = P * nI;
                a.cls_end[1] = a.cls_end[0] + P * 2u * (uint32_t)(mbx - 2);
                a.cls_end[2] = a.cls_end[1] + P * 2u * (uint32_t)(mby - 2);
                a.div_int = make_fastdiv(nI);
                a.div_icols = make_fastdiv((uint32_t)(mbx - 2));
                a.div_rows2 = make_fastdiv(2u * (uint32_t)(mbx - 2));
                a.div_cols2 = make_fastdiv(2u * (uint32_t)(mby - 2));
            }
        }
        // (the streamed-frames variant is a separate instantiation: the flag wait in its move-in
        // costs the device-resident kernel its uniform-datapath index math, 2 % of M4)
        if (range == 32)
            st = ready ? launch_fast<32, kStreamed>(rm, cm, a, nox, total, s) : launch_fast<32, kPlain>(rm, cm, a, nox, total, s);
        else
            st = ready ? launch_fast<16, kStreamed>(rm, cm, a, nox, total, s) : launch_fast<16, kPlain>(rm, cm, a, nox, total, s);
        if (st) return st;
    } else {
        const int smem = a.win * a.win + kMB * kMB;
        {  // the shared-memory attribute is per device: set it once on each
            static std::mutex mu;
            static bool set[kMaxDev] = {};
            int dev = 0;
            SP_CUDA_TRY(cudaGetDevice(&dev));
            if (dev < 0 || dev >= kMaxDev) return SP_ERR_UNSUPPORTED;
            std::lock_guard<std::mutex> lk(mu);
            if (!set[dev]) {
                SP_CUDA_TRY(cudaFuncSetAttribute(me_sad_generic_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                                 142 * 142 + 256));
                set[dev] = true;
            }
        }
        me_sad_generic_kernel<<<dim3(mbx, rows, n_pairs), 256, smem, s>>>(ref, cur, pitch, rows_in_buffer, n_pairs > 1 ? pair_stride : 0, a);
    }
    SP_CUDA_TRY(cudaGetLastError());
    return SP_OK;
}

// Range mode: the macroblocks of flat (pair, MB row) rows [flat_begin, flat_end) of a batch,
// full frames in the buffers (pair p at + (p - pair_base) * pair_stride), outputs indexed
// globally.  gx != nullptr: results also stored into every rank's outputs (fused all-gather).
int me_range_impl(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width, int32_t frame_height,
                  int32_t n_pairs_buffer, int64_t pair_stride, int32_t pair_base, int32_t range, int64_t flat_begin,
                  int64_t flat_end, int16_t* mv, uint32_t* best_sad, void* stream, const GatherArgs* gx) {
    if (!ref || !cur || !mv || !best_sad || (reinterpret_cast<uintptr_t>(mv) & 3) ||
        (reinterpret_cast<uintptr_t>(best_sad) & 3))
        return SP_ERR_INVALID_ARG;
    if (range < 0 || range > 63 || width < kMB || frame_height < kMB || n_pairs_buffer < 0 || pair_base < 0)
        return SP_ERR_INVALID_ARG;
    if (pitch < width || (pitch & 15) || (pair_stride & 15) || (reinterpret_cast<uintptr_t>(ref) & 15) ||
        (reinterpret_cast<uintptr_t>(cur) & 15))
        return SP_ERR_INVALID_ARG;
    if (n_pairs_buffer > 1 && pair_stride < pitch * frame_height) return SP_ERR_INVALID_ARG;
    const int64_t mbx = width / kMB, mby = frame_height / kMB;
    if (flat_begin > flat_end ||
        (flat_end > flat_begin &&
         (flat_begin < (int64_t)pair_base * mby || flat_end > (int64_t)(pair_base + n_pairs_buffer) * mby)))
        return SP_ERR_INVALID_ARG;
    if ((int64_t)(pair_base + n_pairs_buffer) * mby * mbx >= (int64_t(1) << 31)) return SP_ERR_UNSUPPORTED;
    if (gx && !fast_range(range)) return SP_ERR_UNSUPPORTED;
    const cudaStream_t s = (cudaStream_t)stream;
    if (flat_end == flat_begin || mbx == 0) {
        if (!gx) return SP_OK;  // (an empty range still takes part in the gather protocol)
    }
    const int64_t ps = n_pairs_buffer > 1 ? pair_stride : pitch * frame_height;
    if (!fast_range(range)) {
        // generic kernel: one launch per (pair, MB-row band) piece of the range
        for (int64_t f = flat_begin; f < flat_end;) {
            const int64_t p = f / mby, r0 = f % mby, r1 = std::min<int64_t>(mby, r0 + (flat_end - f));
            const int64_t o = (p * mby + r0) * mbx;
            int st = me_search_impl(ref + (p - pair_base) * ps, cur + (p - pair_base) * ps, pitch, width, frame_height,
                                    0, frame_height, 1, ps, kMB, range, (int32_t)r0, (int32_t)r1, mv + 2 * o,
                                    best_sad + o, nullptr, stream, 0);
            if (st) return st;
            f += r1 - r0;
        }
        return SP_OK;
    }
    MeArgs a{width, frame_height, 0, range, n_pairs_buffer, (int32_t)mbx, 0, (int32_t)mby, 2 * range + 16, 0, 0,
             mv, best_sad, nullptr, nullptr, nullptr, (uint32_t)(flat_begin * mbx), pair_base,
             (uint32_t)((flat_end - flat_begin) * mbx), (uint32_t)(flat_end - flat_begin)};
    a.div_per_pair = make_fastdiv((uint32_t)(mby * mbx));
    a.div_mbx = make_fastdiv((uint32_t)mbx);
    int st;
    if ((st = counter_slot(s, &a.counter))) return st;
    CUtensorMap rm, cm;
    const int32_t np = n_pairs_buffer > 0 ? n_pairs_buffer : 1;
    if ((st = cached_map(&rm, ref, width, frame_height, np, pitch, ps, (uint32_t)a.win, (uint32_t)a.win))) return st;
    if ((st = cached_map(&cm, cur, width, frame_height, np, pitch, ps, kMB, kMB))) return st;
    int64_t total = (int64_t)a.total_mb;
    if (gx) {
        if (total == 0) {  // nothing to search: a one-CTA launch still arms and signals the gather
            total = 1;
            a.total_mb = 0;
        }
        st = range == 32 ? launch_fast<32, kGather>(rm, cm, a, *gx, total, s) : launch_fast<16, kGather>(rm, cm, a, *gx, total, s);
    } else {
        const GatherArgs nox{};
        st = range == 32 ? launch_fast<32, kPlain>(rm, cm, a, nox, total, s) : launch_fast<16, kPlain>(rm, cm, a, nox, total, s);
    }
    if (st) return st;
    SP_CUDA_TRY(cudaGetLastError());
    return SP_OK;
}

__global__ void me_gather_wait_kernel(const unsigned long long* done, int32_t nranks, unsigned long long epoch) {
    const int q = threadIdx.x;
    if (q < nranks) {
        const long long t0 = clock64();
        while (ld_acquire_sys(done + q) < epoch) {
            __nanosleep(256);
            if (clock64() - t0 > (40ll << 30)) __trap();  // a rank that never arrives: ~20 s
        }
    }
    __syncthreads();
}

}  // namespace

extern "C" int sp_me_sad_search_range(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                                      int32_t frame_height, int32_t n_pairs_buffer, int64_t pair_stride,
                                      int32_t pair_base, int32_t range, int64_t flat_begin, int64_t flat_end,
                                      int16_t* mv, uint32_t* best_sad, void* stream) {
    SP_NVTX("sp_me_sad_search_range");
    return me_range_impl(ref, cur, pitch, width, frame_height, n_pairs_buffer, pair_stride, pair_base, range,
                         flat_begin, flat_end, mv, best_sad, stream, nullptr);
}

extern "C" int sp_me_sad_search_gather(const sp_me_gather_links* L, const uint8_t* ref, const uint8_t* cur,
                                       int64_t pitch, int32_t width, int32_t frame_height, int32_t n_pairs_buffer,
                                       int64_t pair_stride, int32_t pair_base, int32_t range, int64_t flat_begin,
                                       int64_t flat_end, void* stream) {
    SP_NVTX("sp_me_sad_search_gather");
    if (!L || L->nranks < 1 || L->nranks > SP_ME_MAX_RANKS || L->rank < 0 || L->rank >= L->nranks || L->epoch < 1)
        return SP_ERR_INVALID_ARG;
    static_assert(SP_ME_MAX_RANKS == kMaxGatherRanks, "gather rank limit");
    GatherArgs x{};
    for (int q = 0; q < L->nranks; ++q) {
        if (!L->mv[q] || !L->sad[q] || !L->flags[q]) return SP_ERR_INVALID_ARG;
        x.mv[q] = L->mv[q];
        x.sad[q] = L->sad[q];
        x.flags[q] = L->flags[q];
    }
    x.nranks = L->nranks;
    x.rank = L->rank;
    x.epoch = (unsigned long long)L->epoch;
    int st = me_range_impl(ref, cur, pitch, width, frame_height, n_pairs_buffer, pair_stride, pair_base, range,
                           flat_begin, flat_end, L->mv[L->rank], L->sad[L->rank], stream, &x);
    if (st) return st;
    // the stream continues only when every rank's results have landed in this rank's outputs
    me_gather_wait_kernel<<<1, 32, 0, (cudaStream_t)stream>>>(L->flags[L->rank] + L->nranks, L->nranks, x.epoch);
    SP_CUDA_TRY(cudaGetLastError());
    return SP_OK;
}

extern "C" int sp_me_sad_search(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                                int32_t rows_in_buffer, int32_t row0_global, int32_t frame_height, int32_t n_pairs,
                                int64_t pair_stride, int32_t block, int32_t range, int32_t mb_row_begin,
                                int32_t mb_row_end, int16_t* mv, uint32_t* best_sad, uint32_t* surface, void* stream) {
    SP_NVTX("sp_me_sad_search");
    return me_search_impl(ref, cur, pitch, width, rows_in_buffer, row0_global, frame_height, n_pairs, pair_stride,
                          block, range, mb_row_begin, mb_row_end, mv, best_sad, surface, stream, 0);
}

extern "C" int sp_me_sad_search_unrestricted(const uint8_t* ref_padded, const uint8_t* cur_padded, int64_t pitch,
                                             int32_t width, int32_t height, int32_t pad, int32_t n_pairs,
                                             int64_t pair_stride, int32_t block, int32_t range, int16_t* mv,
                                             uint32_t* best_sad, uint32_t* surface, void* stream) {
    SP_NVTX("sp_me_sad_search_unrestricted");
    if (range < 0 || pad < range || (fast_range(range) && (pad % 16)) || pad < 1) return SP_ERR_INVALID_ARG;
    return me_search_impl(ref_padded, cur_padded, pitch, width, height + 2 * pad, 0, height, n_pairs, pair_stride,
                          block, range, 0, height / kMB, mv, best_sad, surface, stream, pad);
}

namespace {
// A pointer the kernel can store to: device memory as is, page-locked host memory through its
// device mapping.  Pageable host memory is rejected.
int me_device_view(void* p, void** out) {
    cudaPointerAttributes at;
    SP_CUDA_TRY(cudaPointerGetAttributes(&at, p));
    if (at.type == cudaMemoryTypeDevice || at.type == cudaMemoryTypeManaged) {
        *out = p;
        return SP_OK;
    }
    if (at.type == cudaMemoryTypeHost) {
        SP_CUDA_TRY(cudaHostGetDevicePointer(out, p, 0));
        return SP_OK;
    }
    return SP_ERR_INVALID_ARG;
}

// library-owned page-locked constant 1: the source of the ready-flag copies (a stream-ordered
// H2D copy, executed by the copy engine: no SM is needed while the search occupies them all)
const int32_t* pinned_one() {
    static int32_t* one = nullptr;
    static std::once_flag once;
    std::call_once(once, [] {
        void* p = nullptr;
        if (cudaHostAlloc(&p, 64, cudaHostAllocPortable) == cudaSuccess) {
            one = static_cast<int32_t*>(p);
            for (int i = 0; i < 16; ++i) one[i] = 1;  // up to 16 ready flags per copy
        }
    });
    return one;
}

cudaStream_t own_copy_stream() {  // per device (the current one); used when the caller passes no copy stream
    static std::mutex mu;
    static cudaStream_t cs[kMaxDev] = {};
    int dev = 0;
    if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= kMaxDev) return nullptr;
    std::lock_guard<std::mutex> lk(mu);
    if (!cs[dev] && cudaStreamCreateWithFlags(&cs[dev], cudaStreamNonBlocking) != cudaSuccess) cs[dev] = nullptr;
    return cs[dev];
}
}  // namespace

extern "C" int sp_me_search_host(const uint8_t* frames_host, int64_t pitch, int32_t width, int32_t height,
                                 int32_t n_frames, int32_t range, uint8_t* frames_dev, int32_t* ready, int16_t* mv,
                                 uint32_t* best_sad, void* stream, void* copy_stream) {
    SP_NVTX("sp_me_search_host");
    if (!frames_host || !frames_dev || !ready || !mv || !best_sad || n_frames < 1 || height < kMB || width < kMB)
        return SP_ERR_INVALID_ARG;
    if (!fast_range(range)) return SP_ERR_UNSUPPORTED;
    if ((pitch & 15) || pitch < width) return SP_ERR_INVALID_ARG;
    {
        cudaPointerAttributes at;
        SP_CUDA_TRY(cudaPointerGetAttributes(&at, frames_host));
        if (at.type != cudaMemoryTypeHost) return SP_ERR_INVALID_ARG;  // page-locked frames only
    }
    if (n_frames == 1) return SP_OK;
    void *dmv = nullptr, *dsad = nullptr;
    int st;
    if ((st = me_device_view(mv, &dmv)) || (st = me_device_view(best_sad, &dsad))) return st;
    const int32_t* one = pinned_one();
    cudaStream_t cs = copy_stream ? (cudaStream_t)copy_stream : own_copy_stream();
    if (!one || !cs) {
        sp::set_cuda_error((int)cudaErrorMemoryAllocation);
        return SP_ERR_CUDA;
    }
    const cudaStream_t s = (cudaStream_t)stream;
    const size_t fbytes = (size_t)pitch * height;
    const int32_t pairs = n_frames - 1;
    // ready flags cleared in stream order before the copies may set them
    cudaEvent_t ev0, ev1;
    SP_CUDA_TRY(cudaEventCreateWithFlags(&ev0, cudaEventDisableTiming));
    SP_CUDA_TRY(cudaEventCreateWithFlags(&ev1, cudaEventDisableTiming));
    SP_CUDA_TRY(cudaMemsetAsync(ready, 0, (size_t)pairs * sizeof(int32_t), s));
    SP_CUDA_TRY(cudaEventRecord(ev0, s));
    SP_CUDA_TRY(cudaStreamWaitEvent(cs, ev0, 0));
    // The copies are enqueued BEFORE the search is launched: the kernel spins on their flags,
    // so under a serialising tool (ncu, CUDA_LAUNCH_BLOCKING=1) copies enqueued after it would
    // never run — a launch-first order (tried in session 3: 8.54 vs 8.56 ms on M4) deadlocks
    // there until the kernel's trap.
    // frames in groups — the first pair's two frames, then single frames while the search
    // ramps up, then four at a time — each group followed by one copy of the ready flags of
    // the pairs it completes (38 enqueued copies for M4's 65 frames instead of 130: the
    // enqueue sits before the launch)
    for (int32_t f0 = 0; f0 < n_frames;) {
        const int32_t g = f0 == 0 ? 2 : f0 < 5 ? 1 : 4;
        const int32_t f1 = f0 + g < n_frames ? f0 + g : n_frames;
        SP_CUDA_TRY(cudaMemcpyAsync(frames_dev + f0 * fbytes, frames_host + f0 * fbytes, (size_t)(f1 - f0) * fbytes,
                                    cudaMemcpyHostToDevice, cs));
        const int32_t p0 = f0 > 0 ? f0 - 1 : 0, p1 = f1 - 1;  // pairs p0 .. p1-1 now have both frames
        if (p1 > p0)
            SP_CUDA_TRY(cudaMemcpyAsync(ready + p0, one, (size_t)(p1 - p0) * sizeof(int32_t), cudaMemcpyHostToDevice, cs));
        f0 = f1;
    }
    SP_CUDA_TRY(cudaEventRecord(ev1, cs));
    st = me_search_impl(frames_dev, frames_dev + fbytes, pitch, width, height, 0, height, pairs, (int64_t)fbytes, kMB,
                        range, 0, height / kMB, static_cast<int16_t*>(dmv), static_cast<uint32_t*>(dsad), nullptr,
                        stream, 0, ready);
    // the caller's stream completes only after the copies did (frames_dev / ready reusable)
    SP_CUDA_TRY(cudaStreamWaitEvent(s, ev1, 0));
    cudaEventDestroy(ev0);
    cudaEventDestroy(ev1);
    return st;
}

namespace {
__global__ void pad_frames_kernel(const uint8_t* __restrict__ src, int64_t spitch, int64_t sstride, int32_t width,
                                  int32_t height, int32_t pad, uint8_t* __restrict__ dst, int64_t dpitch,
                                  int64_t dstride) {
    const int f = blockIdx.z;
    const int W2 = width + 2 * pad, H2 = height + 2 * pad;
    for (int y = blockIdx.y * blockDim.y + threadIdx.y; y < H2; y += gridDim.y * blockDim.y) {
        const int sy = min(max(y - pad, 0), height - 1);
        const uint8_t* srow = src + (int64_t)f * sstride + (int64_t)sy * spitch;
        uint8_t* drow = dst + (int64_t)f * dstride + (int64_t)y * dpitch;
        for (int x = blockIdx.x * blockDim.x + threadIdx.x; x < W2; x += gridDim.x * blockDim.x)
            drow[x] = srow[min(max(x - pad, 0), width - 1)];
    }
}
}  // namespace

extern "C" int sp_me_pad_frames(const uint8_t* src, int64_t src_pitch, int64_t src_frame_stride, int32_t width,
                                int32_t height, int32_t n_frames, int32_t pad, uint8_t* dst, int64_t dst_pitch,
                                int64_t dst_frame_stride, void* stream) {
    if (!src || !dst || width < 1 || height < 1 || n_frames < 0 || pad < 0 || src_pitch < width ||
        dst_pitch < width + 2 * pad || (n_frames > 1 && (src_frame_stride < src_pitch * height ||
                                                         dst_frame_stride < dst_pitch * (height + 2 * pad))))
        return SP_ERR_INVALID_ARG;
    if (n_frames == 0) return SP_OK;
    dim3 block(128, 4), grid((width + 2 * pad + 127) / 128, 64, n_frames);
    pad_frames_kernel<<<grid, block, 0, (cudaStream_t)stream>>>(src, src_pitch, src_frame_stride, width, height, pad,
                                                               dst, dst_pitch, dst_frame_stride);
    SP_CUDA_TRY(cudaGetLastError());
    return SP_OK;
}

#if SP_ME_EXP & 32
extern "C" int sp_me_cta_read(unsigned long long* out) {
    SP_CUDA_TRY(cudaMemcpyFromSymbol(out, g_me_cta, sizeof(unsigned long long) * 4096 * 3));
    return SP_OK;
}
#endif
#if SP_ME_EXP & 16
// development instrumentation only (tools/me_sections.py): read and reset the section counters
extern "C" int sp_me_prof_read(unsigned long long* out) {
    SP_CUDA_TRY(cudaMemcpyFromSymbol(out, g_me_prof, sizeof(unsigned long long) * 8));
    static const unsigned long long zero[8] = {0, 0, 0, 0, 0, 0, 0, 0};
    SP_CUDA_TRY(cudaMemcpyToSymbol(g_me_prof, zero, sizeof(zero)));
    return SP_OK;
}
#endif

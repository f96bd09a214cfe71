/*
 * sp.h — C ABI of libsp, a B200-native (sm_100a) implementation of the data-parallel
 * hot path of Baskaran, Bondhugula, Krishnamoorthy, Ramanujam, Rountev, Sadayappan,
 * "Automatic Data Movement and Computation Mapping for Multi-level Parallel
 * Architectures with Explicitly Managed Memories", PPoPP'08.
 *
 * Citations "P:Lx-y" are lines of the paper text; "R-xx" are the readings of
 * garbled or silent passages listed in DESIGN.md.
 *
 * Conventions (every entry point):
 *   - plain C types only; every integer is fixed width; no exception crosses the ABI;
 *   - the return value is a status code (SP_OK or a negative SP_ERR_*);
 *   - the caller owns every array and stream; the library never frees caller memory,
 *     keeps no pointer after return, and makes no device allocation on a hot path;
 *   - `stream` arguments are cudaStream_t passed as void* (NULL = legacy default stream);
 *     device entry points are stream-ordered and asynchronous: argument and launch
 *     errors are returned immediately, device faults surface at the caller's next sync;
 *   - there is no CPU fallback: on a machine without a usable sm_100 device the device
 *     entry points return SP_ERR_CUDA.
 */
#ifndef SP_H_
#define SP_H_

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define SP_OK 0
#define SP_ERR_INVALID_ARG -1 /* bad sizes, null required pointer, misalignment */
#define SP_ERR_UNBOUNDED -2   /* planner: a statement domain is unbounded */
#define SP_ERR_CAPACITY -3    /* caller output array too small; required count written back */
#define SP_ERR_OVERFLOW -4    /* int64 overflow in bounds / sizes / coefficients */
#define SP_ERR_UNSUPPORTED -5 /* outside the supported envelope (see each function) */
#define SP_ERR_SMEM_LIMIT -6  /* planner: total staged size exceeds opts->mup_elems */
#define SP_ERR_CUDA -7        /* CUDA error; sp_last_cuda_error() gives the cudaError_t */
#define SP_ERR_NCCL -8        /* NCCL error; sp_last_nccl_error() gives the ncclResult_t */

/* Human-readable name of a status code (static storage). */
const char* sp_status_string(int status);
/* cudaError_t / ncclResult_t of the last failing call on this host thread (0 if none). */
int sp_last_cuda_error(void);
int sp_last_nccl_error(void);
/* Library version, major*10000 + minor*100 + patch. */
int sp_version(void);
/* sizeof of every ABI struct, in this order: sp_domain, sp_ref, sp_block, sp_plan_opts,
 * sp_buffer, sp_jacobi_plan, sp_peer_links, sp_tile_problem, sp_tile_result, sp_op,
 * sp_stmt_body, sp_array_desc, sp_exec_opts, sp_exec_stats.  Writes min(n, 14) entries and
 * returns 14 — lets a binding check its struct layouts against the library's. */
int sp_abi_struct_sizes(int64_t* out, int32_t n);

/* =====================================================================================
 * 1. Planner — the paper's data-management framework for one program block
 *    ("takes as input the iteration spaces of all statements in a program
 *    block as well as the access functions of all array references"; §3.1, Alg. 1,
 *    Alg. 2, §3.1.2, §3.1.3).  Host-only, pure, thread-safe, synchronous.
 * ===================================================================================== */
#define SP_MAX_RANK 8  /* max array dimensionality */
#define SP_MAX_DEPTH 8 /* max loop depth of a statement */
#define SP_MAX_PARAMS 8

/* Iteration-space polytope of a statement (§2): every integer vector i with
 * row . (i, p, 1) >= 0 for each of the n_rows rows; `rows` is row-major
 * [n_rows][depth + n_params + 1].  The domain must be bounded (else SP_ERR_UNBOUNDED). */
typedef struct {
    int32_t depth;
    int32_t n_rows;
    const int64_t* rows;
} sp_domain;

/* Affine array reference A[F . (i, p, 1)] (§2): `rows` is row-major
 * [rank][depth_of_stmt + n_params + 1]; subscript k = rows[k] . (i, p, 1).
 * `array` is a caller-chosen array id; every reference to one array has the same rank. */
typedef struct {
    int32_t stmt;
    int32_t array;
    int32_t is_write;
    int32_t rank;
    const int64_t* rows;
} sp_ref;

typedef struct {
    int32_t n_params;
    int32_t n_stmts;
    int32_t n_refs;
    int32_t reserved;       /* must be 0 */
    const int64_t* params;  /* [n_params] concrete parameter values */
    const sp_domain* stmts; /* [n_stmts] */
    const sp_ref* refs;     /* [n_refs] */
} sp_block;

enum {
    SP_PLAN_PER_ARRAY = 0,  /* one buffer per array: the bounding box of all its data
                               spaces — what Figure 1 prints (reading R-P1) */
    SP_PLAN_COMPONENTS = 1  /* one buffer per connected component of the overlap graph
                               (Alg. 2 step 5) */
};

typedef struct {
    int32_t mode;          /* SP_PLAN_PER_ARRAY or SP_PLAN_COMPONENTS */
    int32_t reuse_filter;  /* 1: stage only partitions Alg. 1 marks beneficial (GPU rule,
                              P:L349-351); refs of other partitions map to -1 */
    double delta;          /* Alg. 1 constant-reuse threshold, 0.30 in the paper */
    int64_t mup_elems;     /* M_up in elements; 0 = unlimited.  If the staged
                              buffers' total size exceeds it: SP_ERR_SMEM_LIMIT */
    int64_t max_points;    /* enumeration budget (integer points over all statements);
                              0 = default 2^27; exceeding it: SP_ERR_UNSUPPORTED */
    int32_t compress;      /* 0: the local array keeps every dimension of the global array
                              (reading R-P5).  1: §3.1.2 literally — a dimension
                              that is an affine function of the earlier dimensions on the
                              partition's data spaces (their affine hull) does not appear in
                              the local array: n = dim of the hull, size = prod over the kept
                              dimensions, F' drops the rows of the others (reading R-P8) */
    int32_t reserved;      /* must be 0 */
} sp_plan_opts;

/* One local-memory buffer = one partition of an array's data spaces (Alg. 2 output). */
typedef struct {
    int32_t array;       /* array id */
    int32_t rank;        /* rank m of the global array; lb / ub / in_* / out_* and the
                            local access rows are given for all m dimensions (n_dims below) */
    int32_t beneficial;  /* Alg. 1 verdict */
    int32_t n_refs;      /* references in the partition */
    int64_t lb[SP_MAX_RANK]; /* lower bound per dimension = offset g */
    int64_t ub[SP_MAX_RANK]; /* upper bound per dimension; empty buffer: lb = 0, ub = -1 */
    int64_t size;            /* prod (ub_k - lb_k + 1) elements */
    int64_t v_in_ub;         /* upper bound on the move-in volume */
    int64_t v_out_ub;        /* upper bound on the move-out volume */
    int64_t in_lb[SP_MAX_RANK], in_ub[SP_MAX_RANK]; /* bbox of the move-in set = union of
                                                       read data spaces */
    int64_t in_count;        /* |union of read data spaces| (0: nothing to move in) */
    int64_t out_lb[SP_MAX_RANK], out_ub[SP_MAX_RANK]; /* bbox of the move-out set */
    int64_t out_count;       /* |union of write data spaces| */
    int32_t in_dense;        /* in_count == volume of the in bbox (a box copy is exact) */
    int32_t out_dense;       /* out_count == volume of the out bbox */
    int64_t overlap;         /* sum over reference pairs of |D_r ∩ D_r'| (Alg. 1 line 7) */
    int64_t union_count;     /* |union of the partition's data spaces| */
    int32_t n_dims;          /* dimensionality n of the local array: = rank, or
                                with compress the dimension of the data spaces' affine hull */
    int32_t kept_mask;       /* bit k set: global dimension k is a dimension of the local
                                array.  Dropped dimensions have local extent 1 and local
                                index 0 (their lb / ub still report the bounding box); the
                                local array is row-major over the kept dimensions in global
                                order, size = prod over kept k of (ub_k - lb_k + 1) */
} sp_buffer;

/* Plan the local buffers of one program block.
 *   bufs[cap_bufs]  : output buffers ordered by (array id, smallest ref index in the
 *                     partition).  If more than cap_bufs are needed, *n_bufs receives the
 *                     required count and SP_ERR_CAPACITY is returned (nothing else written).
 *   ref_buf[n_refs] : buffer index of each reference, -1 if not staged (nullable).
 *   local_rows      : sum over refs of rank x (depth + n_params + 1) int64, in ref order:
 *                     the local access function F' - g; unchanged F for
 *                     unstaged refs (nullable).  Rows of dimensions a buffer does not keep
 *                     (compress) are all zero: local index 0 along an extent-1 axis.
 * Empty statement domains are not errors: they yield empty (size-0) data spaces. */
int sp_plan_buffers(const sp_block* blk, const sp_plan_opts* opts, sp_buffer* bufs, int32_t cap_bufs,
                    int32_t* n_bufs, int32_t* ref_buf, int64_t* local_rows);

/* =====================================================================================
 * 2. Time-tiled 1-D Jacobi
 *
 *   for t in [0, steps): for i in [1, n-2]: a'[i] = ((a[i-1] + a[i]) + a[i+1]) * w
 *   w = fl32(1/3), every operation rounded to nearest fp32, no contraction; a[0] and
 *   a[n-1] are fixed (reading R-J1).
 *
 * Execution: passes of h = min(time_tile, remaining) steps
 * (overlapped "concurrent start" tiling, R-J4); a pass splits [0, n) into space tiles of
 * S cells; a CTA stages each tile's footprint [max(0,x0-H), min(n-1,x0+S-1+H)], H = the
 * time tile rounded up to a multiple of 4, into shared memory (TMA bulk copy), runs the h
 * steps in registers (warp shuffles), and writes back only its owned cells
 * [x0, min(n-1, x0+S-1)] (R-J5).  The kernel boundary is the inter-pass barrier.
 * ===================================================================================== */
typedef struct {
    int64_t n;
    int32_t steps;
    int32_t time_tile;   /* Tt: steps per pass */
    int32_t halo;        /* H: halo cells per side actually staged (Tt rounded up to 4) */
    int32_t passes;      /* ceil(steps / Tt) */
    int64_t space_tile;  /* S: owned cells per tile */
    int64_t tiles;       /* tiles per pass = ceil(n / S) */
    int32_t grid;        /* CTAs per launch (persistent) */
    int32_t threads;     /* threads per CTA */
    int32_t smem_bytes;  /* dynamic shared memory per CTA */
    int32_t cells_per_thread; /* register cells per thread */
    /* the persistent launch over DEVICE memory (sp_jacobi1d_timetiled_fused, _stream with
     * device in / out, sp_jacobi1d_host, the peer-fused launch) uses the in-place geometry
     * when time_tile >= 48 (112 register cells per thread in 57 packed registers, alternating
     * sweeps; with shorter passes the staged geometry is faster); with space_tile = 0 its tile
     * is larger: */
    int64_t persistent_space_tile; /* S of that launch (space_tile if given) */
    int64_t persistent_tiles;      /* its tiles per pass (<= tiles: flags sized by `tiles` suffice) */
} sp_jacobi_plan;

/* Geometry the library will use (host-only).  space_tile = 0 selects the default
 * (largest) tile; otherwise it must be a multiple of 4 not above the default.
 * time_tile in [1, 128].  Errors: SP_ERR_INVALID_ARG. */
int sp_jacobi1d_plan(int64_t n, int32_t steps, int32_t time_tile, int32_t space_tile, sp_jacobi_plan* out);

/* Closed-form footprint of tile (x0, S) in a pass of height h: the Alg. 2 bounding box of
 * the tile's reads of `a`: [max(0, x0-h), min(n-1, x0+S-1+h)]. */
int sp_jacobi1d_tile_footprint(int64_t n, int32_t h, int64_t x0, int64_t space_tile, int64_t* lb, int64_t* ub);

/* Run `steps` steps on device array a[n] (16-byte aligned), using work[n] (16-byte
 * aligned, contents clobbered) as the ping-pong buffer.  On completion a holds a^(steps).
 * n >= 3; steps >= 0 (0 = identity); time_tile in [1, 128]; space_tile 0 or as above.
 * footprint_log (nullable, device int64): [passes][tiles][2] = (lb, ub) of each tile's
 * staged footprint as the kernel computed it (for checking against the planner). */
int sp_jacobi1d_timetiled(float* a, float* work, int64_t n, int32_t steps, int32_t time_tile,
                          int32_t space_tile, int64_t* footprint_log, void* stream);
/* Same result as sp_jacobi1d_timetiled, with every pass in ONE persistent launch (time_tile
 * >= 32; with shorter passes the call runs one launch per pass, which is faster there —
 * SP_JACOBI_FUSED_PERSISTENT=1 keeps the persistent launch): a tile of
 * pass p+1 starts as soon as the tiles of pass p within reach of its halo are done, so pass
 * boundaries cost neither a launch nor a partly-filled last round of tiles (H8's inter-tile
 * synchronisation, done per tile instead of per pass).
 *   flags[flags_len] : caller-owned device int32 scratch, flags_len >= sp_jacobi1d_plan().tiles + 1;
 *                      zeroed by the call (stream-ordered): one completion counter per tile and
 *                      the work counter from which warps take (pass, tile) units in order.
 * passes x tiles must stay below 2^31 (else SP_ERR_UNSUPPORTED).
 * Every CTA of the launch must be co-resident (the grid is the occupancy limit); a tile whose
 * dependences never complete traps after ~20 s instead of hanging.  footprint_log as in
 * sp_jacobi1d_timetiled, laid out [passes][persistent_tiles][2] (sp_jacobi1d_plan).
 * Geometry: the in-place kernel (sp_jacobi_plan.persistent_space_tile): each lane keeps 56
 * packed cell pairs in 57 registers (one 12-warp CTA per SM) and alternates ascending /
 * descending sweeps, so no second register copy is needed; the tile is staged once per warp
 * and stored from registers. */
int sp_jacobi1d_timetiled_fused(float* a, float* work, int32_t* flags, int64_t flags_len, int64_t n, int32_t steps,
                                int32_t time_tile, int32_t space_tile, int64_t* footprint_log, void* stream);

/* General form of the persistent launch: out = J^steps(in).
 *   in, out   : n fp32, 16-byte aligned, device memory OR page-locked host memory
 *               (cudaHostAlloc / cudaHostRegister; pageable memory -> SP_ERR_INVALID_ARG).
 *               Pass 0's move-in reads `in` and the last pass's move-out writes `out`
 *               directly (TMA bulk copies; over PCIe for host memory), so host<->device
 *               transfer is part of the staged movement, overlapped with the other passes.
 *               in may alias out and buf0 (not buf1: pass 0 writes buf1 while later tiles
 *               of pass 0 still read in); out may alias in, buf0 or buf1 (when out is the
 *               array the last pass reads, see below).
 *   buf0, buf1: device scratch of n fp32 each (distinct), ping-pong between passes.
 *   skew      : unit order.  0 = pass-major (all tiles of pass p, then pass p+1);
 *               D > 0 = wavefront: tile t of pass p is scheduled at key t + D p (D a power
 *               of two exceeding ceil(H/S)), so pass p runs D tiles behind pass p-1 — the passes of a
 *               band of tiles follow each other while its data is still in L2, and pass 0's
 *               reads / the last pass's writes stream concurrently with the middle passes;
 *               < 0 = library default (wavefront, D = 512, doubled until it exceeds
 *               ceil(H/S); $SP_JACOBI_SKEW overrides 512).
 *   flags as for sp_jacobi1d_timetiled_fused; passes x tiles < 2^31.
 * If out is the array the last pass reads (e.g. passes == 1 and out == in), the last pass
 * writes buf[passes & 1] and the result is copied to out (stream-ordered). */
int sp_jacobi1d_timetiled_stream(const float* in, float* out, float* buf0, float* buf1, int32_t* flags,
                                 int64_t flags_len, int64_t n, int32_t steps, int32_t time_tile,
                                 int32_t space_tile, int64_t skew, int64_t* footprint_log, void* stream);

/* End-to-end host-buffer call (the public API behind `e2e`): a_host[n] is PAGE-LOCKED host
 * memory holding a^(0); on completion (stream-ordered) it holds a^(steps).  The result is
 * written by the kernel's own last-pass move-out over PCIe (TMA bulk stores into a_host), in
 * the wavefront order of sp_jacobi1d_timetiled_stream.  The input:
 *   flags_len >= sp_jacobi1d_host_flags_len(): moved in by the copy engine — chunks of
 *     SP_JACOBI_HOST_CHUNK cells copied into buf0 on a library-owned side stream while the
 *     kernel already runs, each followed by a ready flag (flags[tiles + 1 + chunk]) that
 *     releases the pass-0 tiles it feeds (the caller's stream waits for the copies before
 *     it completes);
 *   flags_len >= sp_jacobi1d_plan().persistent_tiles + 1 only: read by pass 0's own TMA
 *     move-in straight from a_host.
 * buf0, buf1 as above (distinct device buffers of n cells, contents clobbered).
 * Errors: SP_ERR_INVALID_ARG for pageable or misaligned a_host. */
#define SP_JACOBI_HOST_CHUNK (1 << 21) /* cells per copy-engine input chunk (8 MiB) */
int sp_jacobi1d_host(float* a_host, float* buf0, float* buf1, int32_t* flags, int64_t flags_len, int64_t n,
                     int32_t steps, int32_t time_tile, int32_t space_tile, void* stream);
/* flags_len that selects the copy-engine input of sp_jacobi1d_host (host-only): persistent
 * tiles + 1 + ceil(n / SP_JACOBI_HOST_CHUNK).  Errors: SP_ERR_INVALID_ARG. */
int sp_jacobi1d_host_flags_len(int64_t n, int32_t steps, int32_t time_tile, int32_t space_tile, int64_t* flags_len);

/* Cluster-resident form for small domains (the paper's "fits in the scratchpad" regime,
 * P:L964-1052, Figs. 5 and 7): the whole array is moved in once into the registers of ONE
 * thread-block cluster (up to 16 CTAs x 8 warps), all `steps` run on chip, and it is moved
 * out once.  Warps exchange E-cell halos every E steps (shared memory inside a CTA,
 * distributed shared memory across the cluster, one cluster barrier per exchange): E = 6
 * with 756 owned cells per warp up to 96,768 cells, E = 14 with 1,764 above — the time
 * tile equals the halo.
 *   in, out : device arrays of n fp32 (may alias); n >= 3, steps >= 0.
 * Errors: SP_ERR_UNSUPPORTED if n exceeds sp_jacobi1d_resident_capacity (which reports the
 * largest n the device can hold in one cluster: 16 x 8 x 1764 = 225,792 cells on B200). */
int sp_jacobi1d_resident_capacity(int64_t* max_cells);
int sp_jacobi1d_resident(const float* in, float* out, int64_t n, int32_t steps, void* stream);

/* Segment form (building block of the multi-GPU layer and of its single-GPU loopback
 * test): one pass of height h over a window of the global domain.
 *   src/dst : device arrays holding global cells [g0, g0 + len); dst receives the new
 *             values of the owned cells [own_begin, own_end) only (global indices), which
 *             must satisfy g0 + H <= own_begin (or own_begin == 0 ... cells < 0 do not
 *             exist) and own_end + H <= g0 + len (or own_end == n_global); H is the halo
 *             for time_tile (= h rounded up to 4).  Global cells 0 and n_global-1 are fixed.
 *   g0 and own_begin must be multiples of 4 (16-byte aligned TMA copies). */
int sp_jacobi1d_pass_segment(const float* src, float* dst, int64_t n_global, int64_t g0, int64_t len,
                             int64_t own_begin, int64_t own_end, int32_t h, int32_t time_tile,
                             int32_t space_tile, void* stream);

/* =====================================================================================
 * 3. Full-search motion estimation (Fig. 2 with WS = 16)
 *
 * Macroblocks (bx, by), x0 = 16 bx, y0 = 16 by, bx < floor(width/16); candidates
 * (dx, dy) in [-R, R]^2 valid iff the displaced block lies inside the frame
 * (R-M3); SAD(dx,dy) = sum_{v,u<16} |cur[y0+v][x0+u] - ref[y0+dy+v][x0+dx+u]| (R-M1);
 * best = lexicographic min of (SAD, |dx|+|dy|, dy, dx) over valid candidates (R-M4).
 *
 * Buffers: ref/cur hold rows [row0_global, row0_global + rows_in_buffer) of frames of
 * `frame_height` rows, row pitch `pitch` bytes (multiple of 16), base 16-byte aligned;
 * pair p is at ref + p*pair_stride and cur + p*pair_stride (pair_stride multiple of 16).
 * The band must contain every row a valid candidate of MB rows [mb_row_begin,
 * mb_row_end) reads: [16*mb_row_begin - R, 16*mb_row_end + R) ∩ [0, frame_height).
 * Outputs (device), for pair p, MB row r (relative to mb_row_begin), bx:
 *   mv[((p*rows + r)*mbx + bx)*2 + {0,1}] = (dx, dy)      int16
 *   best_sad[(p*rows + r)*mbx + bx]                        uint32
 *   surface (nullable) [...][(2R+1)^2], entry (dy+R)(2R+1) + (dx+R), 0xFFFFFFFF if invalid
 * block must be 16 (SP_ERR_UNSUPPORTED otherwise); 0 <= range <= 63.
 * ===================================================================================== */
int sp_me_sad_search(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                     int32_t rows_in_buffer, int32_t row0_global, int32_t frame_height, int32_t n_pairs,
                     int64_t pair_stride, int32_t block, int32_t range, int32_t mb_row_begin,
                     int32_t mb_row_end, int16_t* mv, uint32_t* best_sad, uint32_t* surface, void* stream);

/* End-to-end host-buffer search of a frame sequence (the public API behind the ME `e2e`):
 * pairs p = (ref = frame p, cur = frame p+1), p < n_frames - 1, exactly as sp_me_sad_search
 * over the whole frame.
 *   frames_host : PAGE-LOCKED host memory [n_frames][height][pitch] uint8 (pitch multiple of 16)
 *   frames_dev  : device buffer of the same size (staging; contents overwritten)
 *   ready       : device int32 [n_frames - 1] (scratch; cleared by the call)
 *   mv, best_sad: outputs as in sp_me_sad_search for mb rows [0, height/16), in device memory
 *                 or PAGE-LOCKED host memory (the kernel then stores them over PCIe itself)
 *   copy_stream : stream for the H2D frame copies (nullable: a library-owned stream)
 * The frames are copied frame by frame on copy_stream, each copy followed by a copy-engine write
 * of ready[f-1] = 1; the search on `stream` starts at once and the move-in of every macroblock
 * waits for its pair's flag, so the transfer overlaps the search.  `stream` completes after
 * both the search and the copies.  range must be 16 or 32 (SP_ERR_UNSUPPORTED otherwise). */
int sp_me_search_host(const uint8_t* frames_host, int64_t pitch, int32_t width, int32_t height, int32_t n_frames,
                      int32_t range, uint8_t* frames_dev, int32_t* ready, int16_t* mv, uint32_t* best_sad,
                      void* stream, void* copy_stream);

/* Unrestricted motion vectors (reading R-M7): candidates may point
 * outside the frame; out-of-frame reference pixels take the value of the nearest frame pixel
 * (edge extension, as in MPEG-4 / H.264 unrestricted MVs), so all (2R+1)^2 candidates are
 * valid.  ref_padded / cur_padded point at frames edge-extended by `pad` >= R pixels on every
 * side (sp_me_pad_frames), row pitch `pitch` (multiple of 16, >= width + 2 pad), pair p at
 * + p*pair_stride; for R in {16, 32} pad must be a multiple of 16.  Outputs as for
 * sp_me_sad_search over all floor(height/16) macroblock rows. */
int sp_me_sad_search_unrestricted(const uint8_t* ref_padded, const uint8_t* cur_padded, int64_t pitch, int32_t width,
                                  int32_t height, int32_t pad, int32_t n_pairs, int64_t pair_stride, int32_t block,
                                  int32_t range, int16_t* mv, uint32_t* best_sad, uint32_t* surface, void* stream);
/* Edge-extend n_frames frames (width x height, row pitch src_pitch, frame stride
 * src_frame_stride) by `pad` pixels on each side into dst (dst_pitch >= width + 2 pad). */
int sp_me_pad_frames(const uint8_t* src, int64_t src_pitch, int64_t src_frame_stride, int32_t width, int32_t height,
                     int32_t n_frames, int32_t pad, uint8_t* dst, int64_t dst_pitch, int64_t dst_frame_stride,
                     void* stream);

/* Reference window the ME kernel stages for macroblock (bx, by): the Alg. 2 bounding box
 * of ref[y0+dy+v][x0+dx+u] over valid candidates, = [y0-R, y0+15+R] x [x0-R, x0+15+R]
 * clipped to the frame (lb/ub as (row, col)).  Host-only. */
int sp_me_ref_window(int32_t width, int32_t frame_height, int32_t range, int32_t bx, int32_t by,
                     int64_t lb[2], int64_t ub[2]);

/* =====================================================================================
 * 4. Multi-GPU layer (one process per GPU, NCCL over NVLink / NVSwitch)
 * Jacobi is partitioned spatially with a halo of depth H exchanged once per time tile;
 * ME is partitioned by macroblock rows with R-row reference halos (no exchange during
 * the search; results are all-gathered).
 * ===================================================================================== */
typedef struct sp_comm sp_comm;

/* NCCL unique id of the job (rank 0 creates it and broadcasts the 128 bytes). */
int sp_get_unique_id(uint8_t out_id[128]);
/* Collective: create the communicator on `device` (cudaSetDevice is called). */
int sp_comm_init(sp_comm** out, const uint8_t id[128], int32_t nranks, int32_t rank, int32_t device);
int sp_comm_destroy(sp_comm* c);

/* Distributed time-tiled Jacobi over contiguous slabs (NCCL baseline of the fused peer path
 * below).  Rank r owns global cells [x_begin, x_begin + n_local); a_local/work_local hold
 * [x_begin - H, x_begin + n_local + H) (H = halo of time_tile; cells outside [0, n_global)
 * unused), 16-byte aligned, x_begin a multiple of 4.  Per pass: the two edge segments (first /
 * last H owned cells) run first (sp_jacobi1d_pass_segment), then the next pass's halo exchange
 * (grouped ncclSend/ncclRecv of H cells with each neighbour) runs on the communicator's side
 * stream while the interior segment computes on `stream`; the next pass waits for the exchange.
 * Slabs shorter than 3H run whole, exchange after.  The communicator's asynchronous error is
 * checked after every exchange (SP_ERR_NCCL).  On return (stream-ordered) a_local holds the
 * rank's slab of a^(steps) (its halos are stale). */
int sp_jacobi1d_timetiled_dist(sp_comm* c, float* a_local, float* work_local, int64_t n_global,
                               int64_t x_begin, int64_t n_local, int32_t steps, int32_t time_tile,
                               int32_t space_tile, void* stream);

/* Single-GPU loopback transport of the same partitioned pass loop: nranks virtual slabs
 * on the current device (slab r owns [x_begins[r], x_begins[r] + n_locals[r]), slabs tile
 * [0, n_global) in order, each n_local >= H), halos moved with cudaMemcpyAsync instead of
 * NCCL.  Test vehicle for the decomposition on a one-GPU box; layouts as above. */
int sp_jacobi1d_timetiled_loopback(float** a_locals, float** work_locals, int32_t nranks, int64_t n_global,
                                   const int64_t* x_begins, const int64_t* n_locals, int32_t steps,
                                   int32_t time_tile, int32_t space_tile, void* stream);

/* Fused variant: the halo exchange runs inside the pass kernel over peer memory (NVLink P2P
 * or CUDA-IPC mapped pointers) instead of a separate NCCL step.  At the start of pass p the
 * kernel stores this rank's first / last H owned cells straight into the neighbours'
 * current buffers and raises their epoch flags (release, system scope); only the tiles whose
 * footprint reaches into a halo wait (acquire) for this rank's own flags; interior tiles
 * never wait, so the exchange overlaps the interior work tile by tile.  Every rank uses
 * a_local in even and work_local in odd passes (layout as in sp_jacobi1d_timetiled_dist).
 * Flags are monotone epochs: this call uses epoch0+1 .. epoch0+passes; callers advance
 * epoch0 by the pass count between calls (flags start at 0).  flags[2] / flags[3] receive the
 * left / right neighbour's "done with the call" epoch; the first push of a call waits for
 * them (the push targets a buffer the neighbour may still read in its previous call). */
typedef struct {
    float* left_bufs[2];       /* left neighbour's a_local / work_local (mapped), NULL if none */
    float* right_bufs[2];      /* right neighbour's a_local / work_local (mapped) */
    int64_t left_n_local;      /* left neighbour's owned cell count */
    int64_t right_n_local;
    unsigned long long* left_flags;   /* left neighbour's flags[4] (mapped) */
    unsigned long long* right_flags;  /* right neighbour's flags[4] (mapped) */
    unsigned long long* my_flags;     /* own flags[4]: [0] left-halo epoch, [1] right-halo epoch,
                                         [2] left neighbour done, [3] right neighbour done */
    uint64_t epoch0;
} sp_peer_links;
int sp_jacobi1d_timetiled_peer(const sp_peer_links* links, float* a_local, float* work_local, int64_t n_global,
                               int64_t x_begin, int64_t n_local, int32_t steps, int32_t time_tile,
                               int32_t space_tile, void* stream);
/* The same computation in ONE persistent launch per call (no kernel boundary between
 * passes; B200-native form of §8(e)): tiles are ordered by completion flags as in
 * sp_jacobi1d_timetiled_fused, and the halo exchange happens at tile granularity — a slab's
 * edge tiles of pass p wait for the neighbour's epoch (epoch0 + 1 + p) and the last edge
 * tile of each side pushes the new edge cells into the neighbour's buffer and raises its
 * flag, while the interior tiles run on.  flags: device int32 [flags_len >= tiles + 1 +
 * 2 * passes] (tiles = ceil(n_local / space tile)), zeroed by the call; same links, buffer
 * layout and epoch protocol as sp_jacobi1d_timetiled_peer (advance epoch0 by the pass count
 * between calls).  All ranks of a run must use the same entry point. */
/* (Geometry: the in-place kernel of sp_jacobi1d_timetiled_fused, with the peer push.) */
int sp_jacobi1d_timetiled_peer_fused(const sp_peer_links* links, float* a_local, float* work_local, int32_t* flags,
                                     int64_t flags_len, int64_t n_global, int64_t x_begin, int64_t n_local,
                                     int32_t steps, int32_t time_tile, int32_t space_tile, void* stream);

/* Motion estimation sharded over ranks (§8(e) ME row): the batch's flattened (pair, MB row)
 * space [0, n_pairs * mby) is split into contiguous ranges (partition.me_row_ranges, balanced
 * by valid-candidate count); macroblocks are independent FORALL iterations (Fig. 2,
 * P:L860-861 "requiring no synchronization across thread blocks"), so a rank searches its
 * range without any exchange and the results are all-gathered once per batch.
 *
 * sp_me_sad_search_range: the search of one range on this device.
 *   ref, cur       : FULL frames (rows [0, frame_height)), pair p at + (p - pair_base) *
 *                    pair_stride, p in [pair_base, pair_base + n_pairs_buffer); only the rows
 *                    the range reads need to be valid: cur rows [16 r0, 16 r1) and ref rows
 *                    [16 r0 - R, 16 r1 + R) ∩ [0, frame_height) of each pair's MB rows [r0, r1)
 *                    (partition.me_band_rows: the R-row reference halo).
 *   flat_begin/end : the range, pair_base * mby <= flat_begin <= flat_end <= (pair_base +
 *                    n_pairs_buffer) * mby, mby = floor(frame_height / 16).
 *   mv, best_sad   : GLOBAL outputs [n_pairs][mby][mbx](2) as in sp_me_sad_search (mb_row_begin
 *                    = 0): only the range's entries are written.
 * Other arguments and errors as for sp_me_sad_search (any 0 <= range <= 63). */
int sp_me_sad_search_range(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                           int32_t frame_height, int32_t n_pairs_buffer, int64_t pair_stride, int32_t pair_base,
                           int32_t range, int64_t flat_begin, int64_t flat_end, int16_t* mv, uint32_t* best_sad,
                           void* stream);

/* sp_me_sad_search_gather: sp_me_sad_search_range with the all-gather FUSED into the search
 * kernel over peer memory (NVLink P2P / CUDA-IPC mapped pointers): the thread that finishes a
 * macroblock stores its (MV, SAD) into every rank's output arrays, so the gather overlaps the
 * search macroblock by macroblock; the kernel's last CTA then raises done[rank] = epoch in
 * every rank's flags (release, system scope) and a one-CTA wait kernel holds `stream` until
 * this rank's done[q] >= epoch for all q.  At kernel start rank r announces ready[r] = epoch
 * to every rank (its outputs of the previous call are no longer read, by stream order); a
 * macroblock's peer stores wait for every rank's ready.  R must be 16 or 32.
 *   links->mv[q], sad[q]: rank q's global output arrays (mapped; q == rank: own, device);
 *   links->flags[q]     : rank q's u64 flags[2 * nranks] = ready[nranks], done[nranks]
 *                         (zero-initialised, monotone);
 *   links->epoch        : >= 1, strictly increasing per call, the same on every rank.
 * Every rank must call it once per epoch (an empty range included).  A rank that never
 * arrives makes the others trap after ~20 s instead of hanging. */
#define SP_ME_MAX_RANKS 8
typedef struct {
    int32_t nranks, rank;
    int16_t* mv[SP_ME_MAX_RANKS];
    uint32_t* sad[SP_ME_MAX_RANKS];
    unsigned long long* flags[SP_ME_MAX_RANKS];
    uint64_t epoch;
} sp_me_gather_links;
int sp_me_sad_search_gather(const sp_me_gather_links* links, const uint8_t* ref, const uint8_t* cur, int64_t pitch,
                            int32_t width, int32_t frame_height, int32_t n_pairs_buffer, int64_t pair_stride,
                            int32_t pair_base, int32_t range, int64_t flat_begin, int64_t flat_end, void* stream);

/* NCCL baseline of the same gather: the rank's range by sp_me_sad_search_range, then one
 * grouped ncclBroadcast per rank and output array (root q sends its range in place: an
 * all-gather-v into the global arrays) on `stream`.
 *   flat_ranges : host int64 [nranks][2], every rank's [flat_begin, flat_end) (contiguous). */
int sp_me_sad_search_dist(sp_comm* c, const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                          int32_t frame_height, int32_t n_pairs_buffer, int64_t pair_stride, int32_t pair_base,
                          int32_t range, const int64_t* flat_ranges, int16_t* mv, uint32_t* best_sad, void* stream);

/* Exportable device allocations and CUDA-IPC handles (64 bytes) for the peer path. */
int sp_device_alloc(void** ptr, int64_t bytes); /* cudaMalloc + zero fill */
int sp_device_free(void* ptr);
int sp_ipc_get_handle(const void* ptr, uint8_t out_handle[64]);
int sp_ipc_open_handle(const uint8_t handle[64], void** ptr);
int sp_ipc_close_handle(void* ptr);

/* Failure detection: the communicator's asynchronous NCCL state
 * (ncclCommGetAsyncError; ncclSuccess = 0, ncclInProgress = 7, anything else = the
 * communicator failed and must be destroyed).  Host call, does not synchronize. */
int sp_comm_async_error(sp_comm* c, int32_t* nccl_result);
/* Wait for `stream` with a deadline while polling the communicator's asynchronous error; on
 * an NCCL error, or when timeout_ms elapses first (a peer died or hangs), the communicator
 * is aborted (ncclCommAbort) and SP_ERR_NCCL returned (sp_last_nccl_error: the NCCL result,
 * ncclInProgress = 7 for the timeout); the comm must then only be destroyed.  Host call. */
int sp_comm_sync(sp_comm* c, void* stream, int64_t timeout_ms);

/* ncclAllGather of `bytes` per rank (device buffers) — used for the ME results. */
int sp_allgather(sp_comm* c, const void* send, void* recv, int64_t bytes, void* stream);

/* =====================================================================================
 * 6. Tile-size search (§4.3).  Minimise the paper's
 *    data-movement cost over a grid of candidate tile vectors t (one list per loop):
 *      C(t) = sum_{k in I} prod_{i<=r_k} ceil(N_i/t_i) (P S + V_in_k(t) L / P)
 *           + sum_{k in O} prod_{i<=r_k} ceil(N_i/t_i) (P S + V_out_k(t) L / P)
 *    subject to 0 < t_i <= N_i, sum_k M_k(t) <= M_up, prod t_i >= P.  The tile
 *    is the box 0 <= i_l < t_l of a perfectly nested band; M_k, V_in_k, V_out_k come from
 *    Alg. 2 (sp_plan_buffers, PER_ARRAY) on that box; r_k is the deepest loop array k's
 *    references depend on (movement hoisted above redundant loops, §4.2).  The paper
 *    solves the real relaxation by SQP and rounds; this evaluates the exact
 *    objective on the grid.  Host-only.
 * ===================================================================================== */
typedef struct {
    int32_t depth;          /* m: loops of the band, outermost first (<= SP_MAX_DEPTH) */
    int32_t n_refs;
    const int64_t* extent;  /* [m] N_i (loop trip counts) */
    const sp_ref* refs;     /* rows [rank][m + 1] over the tile-local iterators (stmt ignored) */
    const int32_t* n_cand;  /* [m] number of candidate sizes per loop */
    const int64_t* cand;    /* concatenated candidate sizes (each in [1, N_i]) */
    int64_t mup_elems;      /* M_up in elements; 0 = unlimited */
    int32_t procs;          /* P: inner-level parallel processes per outer process */
    int32_t reserved;       /* must be 0 */
    double sync_cost;       /* S: synchronisation cost per process per movement */
    double elem_cost;       /* L: cost of moving one element */
} sp_tile_problem;

typedef struct {
    int64_t tile[SP_MAX_DEPTH]; /* argmin t */
    double cost;                /* C(t) */
    int64_t local_elems;        /* sum_k M_k(t) */
    int64_t evaluated;          /* candidates evaluated (prod t_i >= P) */
    int32_t feasible;           /* 0: no candidate met the constraints */
    int32_t reserved;
} sp_tile_result;

int sp_tile_search(const sp_tile_problem* prob, sp_tile_result* out);

/* =====================================================================================
 * 5. Ablation baselines: the paper's "GPU w/o scratchpad memory"
 *    versions (Figs. 4-5), same arithmetic and results, no on-chip staging.
 * ===================================================================================== */
/* Jacobi without staging or time tiling: one launch per time step, operands read from
 * global memory.  Same contract as sp_jacobi1d_timetiled (a, work device, n >= 3). */
int sp_jacobi1d_untiled(float* a, float* work, int64_t n, int32_t steps, void* stream);
/* ME without staging: one CTA per macroblock, candidates read straight from global memory.
 * Same arguments and outputs as sp_me_sad_search; pitch, bases and pair_stride need only
 * 4-byte alignment. */
int sp_me_sad_search_direct(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                            int32_t rows_in_buffer, int32_t row0_global, int32_t frame_height, int32_t n_pairs,
                            int64_t pair_stride, int32_t block, int32_t range, int32_t mb_row_begin,
                            int32_t mb_row_end, int16_t* mv, uint32_t* best_sad, uint32_t* surface, void* stream);

/* =====================================================================================
 * 6. Generic staged-tile executor: runs an arbitrary small affine
 *    program block on the GPU exactly as the framework prescribes — local buffers from
 *    sp_plan_buffers (PER_ARRAY bounding boxes, Alg. 2 / Figure 1),
 *    accesses rewritten to the local access functions F'(y) - g, move-in
 *    of the read data spaces before and move-out of the written data spaces after the
 *    block, tiles mapped to CTAs (outer-level parallel units,
 *    §5) and consecutive tiles of one CTA sharing a buffer whose movement is
 *    hoisted out of the tile loop when its data spaces do not change (§4.2).
 *    Inner-level parallelism: statement instances of a tile are grouped into dependence
 *    levels (exact flow/anti/output dependences between instances, computed on the host
 *    in original program order); the CTA's threads run one level at a time.
 * ===================================================================================== */
enum { SP_OP_LOAD = 0, SP_OP_CONST = 1, SP_OP_ADD = 2, SP_OP_SUB = 3, SP_OP_MUL = 4 };
/* One postfix instruction of a statement's right-hand side (fp32, round to nearest, no
 * contraction).  SP_OP_LOAD pushes the value of read reference `ref` (index into
 * blk->refs; must belong to the statement and have is_write = 0); SP_OP_CONST pushes
 * `value`; ADD/SUB/MUL pop b, a and push a op b.  Stack depth <= 16. */
typedef struct {
    int32_t op;
    int32_t ref;
    float value;
    int32_t reserved;
} sp_op;
/* Body of statement s (the paper prints statement bodies only as S1, S2; Figure 1 gives
 * A[i][j+1] = A[i+j][j+1]*3 and B[i][j+k] = A[i][k] + B[i+j][k]). */
typedef struct {
    int32_t write_ref;    /* the statement's write reference (is_write = 1) */
    int32_t n_ops;
    const sp_op* ops;     /* [n_ops] postfix program of the right-hand side */
    const int32_t* beta;  /* [depth + 1] textual positions: instances execute in the
                             lexicographic order of (beta_0, i_0, beta_1, ..., i_{d-1}, beta_d),
                             the original program order (2d+1 schedule) */
} sp_stmt_body;
/* Global array `id` (the sp_ref.array ids index this table): fp32, row-major, device memory. */
typedef struct {
    float* data;
    int32_t rank;
    int32_t reserved;
    int64_t extent[SP_MAX_RANK];
} sp_array_desc;
typedef struct {
    int32_t n_tiles;             /* the block is instantiated once per tile ... */
    int32_t tiles_per_cta;       /* ... and consecutive groups of tiles run in one CTA, in order */
    const int64_t* tile_params;  /* [n_tiles][blk->n_params]: the parameter values of each
                                    tile (NULL with n_tiles = 1: blk->params) */
    int32_t hoist;               /* 1: a buffer whose read and write data spaces are identical
                                    for consecutive tiles of a CTA stays resident (moved in
                                    before the first, out after the last), §4.2 */
    int32_t reuse_filter;        /* 1: stage only what Alg. 1 marks beneficial; other
                                    references access global memory directly */
    int64_t max_points;          /* planner enumeration budget (0 = default) */
    int32_t movement;            /* SP_MOVE_ALL or SP_MOVE_DATAFLOW (below) */
    int32_t dry_run;             /* 1: compile only (stats, move_counts), launch nothing */
    const int32_t* live_out;     /* [n_arrays] (nullable = all 1): SP_MOVE_DATAFLOW writes back
                                    a final value only for live-out arrays */
    int64_t* move_counts;        /* nullable [n_tiles][n_arrays][2]: elements moved in / out */
    int32_t compress;            /* planner option (sp_plan_opts.compress): local buffers drop
                                    affinely dependent dimensions (§3.1.2) */
    int32_t reserved;            /* must be 0 */
} sp_exec_opts;
/* Data movement of a tile (P:L397-405 default; §3.1.4 P:L450-482 optimised):
 *   SP_MOVE_ALL      every element of the read data spaces in, of the write data spaces out;
 *   SP_MOVE_DATAFLOW with the tiles in order as the program: in = elements the tile reads
 *                    before writing them itself; out = elements whose last write in the tile
 *                    is read by a later tile before being rewritten, or that no later tile
 *                    rewrites while their array is live-out (the paper's stated future work,
 *                    realised exactly on statement instances).  Hoisting is not combined
 *                    with it (hoist is ignored). */
enum { SP_MOVE_ALL = 0, SP_MOVE_DATAFLOW = 1 };
typedef struct {
    int64_t instances;           /* statement instances executed */
    int64_t moved_in;            /* elements moved global -> shared */
    int64_t moved_out;           /* elements moved shared -> global */
    int64_t moves_hoisted;       /* element moves saved by hoisting */
    int32_t max_levels;          /* most dependence levels in one tile */
    int32_t smem_bytes;          /* dynamic shared memory per CTA */
    int32_t ctas;                /* CTAs launched */
    int32_t reserved;
} sp_exec_stats;
/* Execute the block.  Tiles in different CTAs must be independent (the caller's FORALL);
 * tiles of one CTA may depend on each other (they run in order).  Every accessed element
 * must lie inside its array's extents (else SP_ERR_INVALID_ARG); the staged buffers of a
 * CTA must fit in shared memory (else SP_ERR_SMEM_LIMIT).  Compiles the per-CTA programs
 * on the host (synchronous), then launches one kernel on `stream`; the compiled program
 * lives in device memory allocated and freed stream-ordered (cudaMallocAsync /
 * cudaFreeAsync) — this is a tool entry point, not a hot path.  stats is nullable. */
int sp_exec_block(const sp_block* blk, const sp_stmt_body* bodies, const sp_array_desc* arrays, int32_t n_arrays,
                  const sp_exec_opts* opts, sp_exec_stats* stats, void* stream);

#ifdef __cplusplus
}
#endif
#endif /* SP_H_ */

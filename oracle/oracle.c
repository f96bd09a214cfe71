/*
 * oracle.c — plain, slow, obviously-correct CPU reference for the two workloads of
 * Baskaran et al., PPoPP'08 (P = /root/reference/PAPER.md).
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load this library.  It shares no code,
 * header, table or constant generator with the CUDA path (paper_conf_..._b200/csrc).
 *
 * Build: gcc -O2 -fopenmp -ffp-contract=off -fno-fast-math -shared -fPIC
 *        (no FMA contraction, no reassociation: every float operation below is rounded
 *        exactly as written).  OpenMP parallelises only over independent outputs
 *        (cells of one time step; macroblocks), so results do not depend on threads.
 *
 * Functions
 *   spo_jacobi1d           — untiled Jacobi, the definition (DESIGN.md R-J1..R-J5).
 *   spo_jacobi1d_tiled     — overlapped time-tiled twin (self-check of the tiling
 *                            argument only; never compared to itself).
 *   spo_jacobi1d_points    — a^(T)_i at chosen i by light-cone windows (sampled parity).
 *   spo_jacobi1d_f64       — the same recurrence in double precision (pins vs closed form).
 *   spo_me_search          — exhaustive full-search SAD motion estimation (R-M1..R-M6).
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#ifdef _OPENMP
#include <omp.h>
#endif

/* ---------------------------------------------------------------------------------
 * Threads
 * ------------------------------------------------------------------------------- */
void spo_set_threads(int n) {
#ifdef _OPENMP
    if (n > 0) omp_set_num_threads(n);
#else
    (void)n;
#endif
}

int spo_get_threads(void) {
#ifdef _OPENMP
    return omp_get_max_threads();
#else
    return 1;
#endif
}

/* ---------------------------------------------------------------------------------
 * 1-D Jacobi ("1-D Jacobi kernel", P:L960-967 time loop around a space
 * loop).  The paper never prints the statement; reading R-J1:
 *   for t in [0, T): for i in [1, N-2]:  b[i] = ((a[i-1] + a[i]) + a[i+1]) * w;  a = b
 * with w = fl32(1/3) and a[0], a[N-1] fixed (Dirichlet).  Implemented with two arrays
 * and a swap, equivalent to the copy-back form.
 * ------------------------------------------------------------------------------- */
static const float SPO_W = 1.0f / 3.0f; /* rounds to 0x3EAAAAAB */

/* In place: on return a holds a^(T).  work must hold n floats. */
void spo_jacobi1d(float* a, int64_t n, int32_t steps, float* work) {
    if (n < 3 || steps <= 0) return;
    float* src = a;
    float* dst = work;
    for (int32_t t = 0; t < steps; ++t) {
        dst[0] = src[0];
        dst[n - 1] = src[n - 1];
#pragma omp parallel for schedule(static)
        for (int64_t i = 1; i < n - 1; ++i) {
            float s = src[i - 1] + src[i];
            s = s + src[i + 1];
            dst[i] = s * SPO_W;
        }
        float* tmp = src; src = dst; dst = tmp;
    }
    if (src != a) memcpy(a, src, (size_t)n * sizeof(float));
}

/* Same recurrence in fp64 with w = 1/3 (double); used only by the closed-form pin. */
void spo_jacobi1d_f64(double* a, int64_t n, int32_t steps, double* work) {
    if (n < 3 || steps <= 0) return;
    const double w = 1.0 / 3.0;
    double* src = a;
    double* dst = work;
    for (int32_t t = 0; t < steps; ++t) {
        dst[0] = src[0];
        dst[n - 1] = src[n - 1];
#pragma omp parallel for schedule(static)
        for (int64_t i = 1; i < n - 1; ++i) dst[i] = ((src[i - 1] + src[i]) + src[i + 1]) * w;
        double* tmp = src; src = dst; dst = tmp;
    }
    if (src != a) memcpy(a, src, (size_t)n * sizeof(double));
}

/* Overlapped time tiling ("concurrent start", DESIGN.md R-J4): for each
 * pass of height h = min(Tt, remaining) and each space tile [x0, x0+S):
 *   1. copy the footprint [max(0,x0-h), min(N-1,x0+S-1+h)] into a local buffer
 *      (Alg. 2 bounding box of the tile's data spaces);
 *   2. run h steps on local cells, keeping global cells 0 and N-1 fixed;
 *   3. write back only [x0, min(N-1, x0+S-1)] (owned region, DESIGN.md R-J5).
 * Must equal spo_jacobi1d bit for bit.  local must hold 2*(S + 2*Tt) floats. */
void spo_jacobi1d_tiled(float* a, int64_t n, int32_t steps, int32_t tt, int64_t s,
                        float* work, float* local) {
    if (n < 3 || steps <= 0 || tt <= 0 || s <= 0) return;
    float* src = a;
    float* dst = work;
    int32_t done = 0;
    while (done < steps) {
        int32_t h = steps - done < tt ? steps - done : tt;
        for (int64_t x0 = 0; x0 < n; x0 += s) {
            int64_t lb = x0 - h < 0 ? 0 : x0 - h;
            int64_t ub = x0 + s - 1 + h > n - 1 ? n - 1 : x0 + s - 1 + h;
            int64_t len = ub - lb + 1;
            float* L0 = local;
            float* L1 = local + len;
            for (int64_t j = 0; j < len; ++j) L0[j] = src[lb + j];
            for (int32_t t = 0; t < h; ++t) {
                for (int64_t j = 0; j < len; ++j) {
                    int64_t g = lb + j;
                    if (g == 0 || g == n - 1 || j == 0 || j == len - 1) {
                        L1[j] = L0[j]; /* boundary cell, or tile edge (stale; never owned) */
                    } else {
                        float v = L0[j - 1] + L0[j];
                        v = v + L0[j + 1];
                        L1[j] = v * SPO_W;
                    }
                }
                float* tmp = L0; L0 = L1; L1 = tmp;
            }
            int64_t oe = x0 + s - 1 > n - 1 ? n - 1 : x0 + s - 1;
            for (int64_t g = x0; g <= oe; ++g) dst[g] = L0[g - lb];
        }
        float* tmp = src; src = dst; dst = tmp;
        done += h;
    }
    if (src != a) memcpy(a, src, (size_t)n * sizeof(float));
}

/* a^(T)_i for m chosen indices, each from the light-cone window [i-T, i+T] ∩ [0, N-1]
 * of a^(0) (a^(T)_i depends only on a^(0)_{i-T..i+T}).  Window edges that are not
 * domain boundaries are held fixed: their error travels one cell per step and reaches
 * cell i only after T+1 steps.  scratch must hold 2*(2T+1) floats. */
void spo_jacobi1d_points(const float* a0, int64_t n, int32_t steps, const int64_t* idx, int64_t m,
                         float* out, float* scratch) {
    for (int64_t q = 0; q < m; ++q) {
        int64_t i = idx[q];
        int64_t lb = i - steps < 0 ? 0 : i - steps;
        int64_t ub = i + steps > n - 1 ? n - 1 : i + steps;
        int64_t len = ub - lb + 1;
        float* L0 = scratch;
        float* L1 = scratch + len;
        for (int64_t j = 0; j < len; ++j) L0[j] = a0[lb + j];
        for (int32_t t = 0; t < steps; ++t) {
            for (int64_t j = 0; j < len; ++j) {
                int64_t g = lb + j;
                if (g == 0 || g == n - 1 || j == 0 || j == len - 1) {
                    L1[j] = L0[j];
                } else {
                    float v = L0[j - 1] + L0[j];
                    v = v + L0[j + 1];
                    L1[j] = v * SPO_W;
                }
            }
            float* tmp = L0; L0 = L1; L1 = tmp;
        }
        out[q] = L0[i - lb];
    }
}

/* h steps of the definition on a window w[0..len) holding global cells [g0, g0+len) of a
 * domain of n cells: global cells 0 and n-1 stay fixed, and so do the window's two edge
 * cells (their true neighbours are outside the window, so after h steps only cells at
 * distance >= h from a non-domain window edge are exact).  scratch: len floats. */
void spo_jacobi1d_window(float* w, int64_t len, int64_t g0, int64_t n, int32_t steps, float* scratch) {
    float* L0 = w;
    float* L1 = scratch;
    for (int32_t t = 0; t < steps; ++t) {
        for (int64_t j = 0; j < len; ++j) {
            int64_t g = g0 + j;
            if (g <= 0 || g >= n - 1 || j == 0 || j == len - 1) {
                L1[j] = L0[j];
            } else {
                float v = L0[j - 1] + L0[j];
                v = v + L0[j + 1];
                L1[j] = v * SPO_W;
            }
        }
        float* tmp = L0; L0 = L1; L1 = tmp;
    }
    if (L0 != w) memcpy(w, L0, (size_t)len * sizeof(float));
}

/* ---------------------------------------------------------------------------------
 * Motion estimation: full search (Fig. 2 nest with WS = 16).
 * DESIGN.md readings R-M1..R-M6:
 *   macroblocks (bx, by), bx < floor(W/16), by < floor(H/16); x0 = 16 bx, y0 = 16 by;
 *   candidates (dx, dy) in [-R, R]^2, valid iff the displaced 16x16 block lies inside
 *   the reference frame;
 *   SAD(dx,dy) = sum_{v,u<16} |cur[y0+v][x0+u] - ref[y0+dy+v][x0+dx+u]|;
 *   best = lexicographic min of (SAD, |dx|+|dy|, dy, dx) over valid candidates.
 * Frames are row-major uint8 with row pitch `pitch` bytes.
 * Outputs for each listed macroblock q (mb index = by * MBX + bx):
 *   mv[2q] = dx, mv[2q+1] = dy; sad[q]; surface (nullable) [(2R+1)^2] per MB with
 *   entry (dy+R)*(2R+1) + (dx+R), 0xFFFFFFFF for invalid candidates.
 * ------------------------------------------------------------------------------- */
static int spo_iabs(int v) { return v < 0 ? -v : v; }

void spo_me_search(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                   int32_t height, int32_t range, const int32_t* mbs, int64_t n_mbs,
                   int16_t* mv, uint32_t* sad, uint32_t* surface) {
    const int B = 16;
    const int mbx = width / B;
    const int side = 2 * range + 1;
#pragma omp parallel for schedule(dynamic, 4)
    for (int64_t q = 0; q < n_mbs; ++q) {
        int bx = mbs[q] % mbx;
        int by = mbs[q] / mbx;
        int x0 = B * bx, y0 = B * by;
        int found = 0;
        uint32_t best_sad = 0;
        int best_dx = 0, best_dy = 0;
        for (int dy = -range; dy <= range; ++dy) {
            for (int dx = -range; dx <= range; ++dx) {
                int valid = (x0 + dx >= 0) && (x0 + dx + B <= width) &&
                            (y0 + dy >= 0) && (y0 + dy + B <= height);
                uint32_t s = 0xFFFFFFFFu;
                if (valid) {
                    s = 0;
                    for (int v = 0; v < B; ++v) {
                        const uint8_t* c = cur + (int64_t)(y0 + v) * pitch + x0;
                        const uint8_t* r = ref + (int64_t)(y0 + dy + v) * pitch + (x0 + dx);
                        for (int u = 0; u < B; ++u) s += (uint32_t)spo_iabs((int)c[u] - (int)r[u]);
                    }
                    int better;
                    if (!found) {
                        better = 1;
                    } else if (s != best_sad) {
                        better = s < best_sad;
                    } else {
                        int l1 = spo_iabs(dx) + spo_iabs(dy);
                        int bl1 = spo_iabs(best_dx) + spo_iabs(best_dy);
                        if (l1 != bl1) better = l1 < bl1;
                        else if (dy != best_dy) better = dy < best_dy;
                        else better = dx < best_dx;
                    }
                    if (better) {
                        found = 1;
                        best_sad = s;
                        best_dx = dx;
                        best_dy = dy;
                    }
                }
                if (surface) surface[q * (int64_t)side * side + (int64_t)(dy + range) * side + (dx + range)] = s;
            }
        }
        /* dx = dy = 0 is always valid, so found == 1 */
        mv[2 * q] = (int16_t)best_dx;
        mv[2 * q + 1] = (int16_t)best_dy;
        sad[q] = best_sad;
    }
}

/* Unrestricted-MV full search (reading R-M7): every candidate (dx, dy) in
 * [-R, R]^2 is valid; reference pixels outside the frame take the value of the nearest
 * frame pixel (edge extension: coordinates clamped to [0, W-1] x [0, H-1]).  Same outputs
 * and tie-break as spo_me_search. */
static int spo_clampi(int v, int lo, int hi) { return v < lo ? lo : (v > hi ? hi : v); }

void spo_me_search_unrestricted(const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width, int32_t height,
                                int32_t range, const int32_t* mbs, int64_t n_mbs, int16_t* mv, uint32_t* sad,
                                uint32_t* surface) {
    const int B = 16;
    const int mbx = width / B;
    const int side = 2 * range + 1;
#pragma omp parallel for schedule(dynamic, 4)
    for (int64_t q = 0; q < n_mbs; ++q) {
        int x0 = B * (mbs[q] % mbx), y0 = B * (mbs[q] / mbx);
        int found = 0, best_dx = 0, best_dy = 0;
        uint32_t best_sad = 0;
        for (int dy = -range; dy <= range; ++dy) {
            for (int dx = -range; dx <= range; ++dx) {
                uint32_t s = 0;
                for (int v = 0; v < B; ++v) {
                    const uint8_t* c = cur + (int64_t)(y0 + v) * pitch + x0;
                    const uint8_t* r = ref + (int64_t)spo_clampi(y0 + dy + v, 0, height - 1) * pitch;
                    for (int u = 0; u < B; ++u)
                        s += (uint32_t)spo_iabs((int)c[u] - (int)r[spo_clampi(x0 + dx + u, 0, width - 1)]);
                }
                int better;
                if (!found) better = 1;
                else if (s != best_sad) better = s < best_sad;
                else {
                    int l1 = spo_iabs(dx) + spo_iabs(dy), bl1 = spo_iabs(best_dx) + spo_iabs(best_dy);
                    if (l1 != bl1) better = l1 < bl1;
                    else if (dy != best_dy) better = dy < best_dy;
                    else better = dx < best_dx;
                }
                if (better) {
                    found = 1;
                    best_sad = s;
                    best_dx = dx;
                    best_dy = dy;
                }
                if (surface) surface[q * (int64_t)side * side + (int64_t)(dy + range) * side + (dx + range)] = s;
            }
        }
        mv[2 * q] = (int16_t)best_dx;
        mv[2 * q + 1] = (int16_t)best_dy;
        sad[q] = best_sad;
    }
}

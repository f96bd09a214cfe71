// planner.cpp — sp_plan_buffers: the paper's automatic data-management framework for
// one program block (P = PAPER.md §3.1, Algorithm 1, Algorithm 2 P:L309-332,
// local access functions §3.1.2, data movement §3.1.3).
//
// B200-era replacement for the paper's toolchain (PIP / CLooG / PolyLib, P:L355-359,
// L373-375, L443-446), specialised to concrete parameter values:
//   * loop bounds for scanning each statement's polytope come from Fourier-Motzkin
//     projection with integer tightening (the CLooG role);
//   * integer points are scanned level by level; at the innermost level the original
//     constraints are applied, so exactly the integer points of the domain are visited;
//   * a data space (the image F . I) is the sorted set of linearised
//     coordinates of the images; set unions / intersections are merges (the PolyLib role);
//   * the bounds lb/ub of a partition are the exact integer min/max over its union, which
//     equal the bounds of its convex hull (bbox(hull) = bbox(union)).
#include <algorithm>
#include <cstdint>
#include <cstring>
#include <numeric>
#include <vector>

#include "../../include/sp.h"
#include "sp_internal.h"

namespace {

using i64 = int64_t;
using i128 = __int128;

constexpr i64 kDefaultMaxPoints = i64(1) << 27;

struct PlanError {
    int code;
};

inline i64 floor_div(i64 a, i64 b) {  // b > 0
    i64 q = a / b;
    if ((a % b != 0) && (a < 0)) --q;
    return q;
}
inline i64 ceil_div(i64 a, i64 b) {  // b > 0
    i64 q = a / b;
    if ((a % b != 0) && (a > 0)) ++q;
    return q;
}
inline i64 to_i64(i128 v) {
    if (v > (i128)INT64_MAX || v < (i128)INT64_MIN) throw PlanError{SP_ERR_OVERFLOW};
    return (i64)v;
}
inline i64 gcd64(i64 a, i64 b) {
    a = a < 0 ? -a : a;
    b = b < 0 ? -b : b;
    while (b) {
        i64 t = a % b;
        a = b;
        b = t;
    }
    return a;
}

// A constraint sum_k c[k] x_k + c[d] >= 0 over the statement's d loop variables
// (parameters already substituted).
using Row = std::vector<i64>;

// Divide by the gcd g of the variable coefficients; the constant is floored, which keeps
// every integer point and removes rational slivers (integer tightening).
bool normalize(Row& r, int d) {
    i64 g = 0;
    for (int k = 0; k < d; ++k) g = gcd64(g, r[k]);
    if (g == 0) return r[d] >= 0;  // constant constraint: feasible iff const >= 0
    if (g > 1) {
        for (int k = 0; k < d; ++k) r[k] /= g;
        r[d] = floor_div(r[d], g);
    }
    return true;
}

struct Scan {
    int d = 0;
    bool empty = false;
    // level L: constraints with a nonzero coefficient on x_L, over x_0..x_L
    std::vector<std::vector<Row>> lower, upper;
};

Scan build_scan(std::vector<Row> sys, int d) {
    Scan s;
    s.d = d;
    s.lower.assign(d, {});
    s.upper.assign(d, {});
    // normalise, drop trivially-true constant rows, detect contradictions
    auto clean = [&](std::vector<Row>& v) -> bool {
        std::vector<Row> out;
        for (auto& r : v) {
            bool allzero = true;
            for (int k = 0; k < d; ++k) allzero &= (r[k] == 0);
            if (allzero) {
                if (r[d] < 0) return false;
                continue;
            }
            if (!normalize(r, d)) return false;
            out.push_back(r);
        }
        std::sort(out.begin(), out.end());
        out.erase(std::unique(out.begin(), out.end()), out.end());
        v.swap(out);
        return true;
    };
    if (!clean(sys)) {
        s.empty = true;
        return s;
    }
    for (int L = d - 1; L >= 0; --L) {
        std::vector<Row> pos, neg, zero;
        for (auto& r : sys) {
            if (r[L] > 0) pos.push_back(r);
            else if (r[L] < 0) neg.push_back(r);
            else zero.push_back(r);
        }
        s.lower[L] = pos;
        s.upper[L] = neg;
        if (L == 0) break;
        // eliminate x_L (Fourier-Motzkin)
        std::vector<Row> next = zero;
        for (auto& p : pos)
            for (auto& n : neg) {
                Row r(d + 1);
                i64 a = p[L], b = -n[L];
                for (int k = 0; k <= d; ++k) r[k] = to_i64((i128)b * p[k] + (i128)a * n[k]);
                r[L] = 0;
                next.push_back(r);
            }
        if (!clean(next)) {
            s.empty = true;
            return s;
        }
        if (next.size() > 20000) throw PlanError{SP_ERR_UNSUPPORTED};
        sys.swap(next);
    }
    for (int L = 0; L < d; ++L)
        if (s.lower[L].empty() || s.upper[L].empty()) throw PlanError{SP_ERR_UNBOUNDED};
    return s;
}

// Visit every integer point of the domain; f(x) receives the loop vector.
template <class F>
void scan_points(const Scan& s, i64 max_points, i64& budget_used, F&& f) {
    if (s.empty) return;
    const int d = s.d;
    i64 x[SP_MAX_DEPTH + 1] = {0};
    if (d == 0) {
        if (++budget_used > max_points) throw PlanError{SP_ERR_UNSUPPORTED};
        f(x);
        return;
    }
    i64 hi[SP_MAX_DEPTH];
    auto bounds = [&](int L, i64& lo, i64& up) {
        lo = INT64_MIN;
        up = INT64_MAX;
        for (auto& r : s.lower[L]) {  // r[L] x_L + rest >= 0  ->  x_L >= ceil(-rest / r[L])
            i128 rest = r[d];
            for (int k = 0; k < L; ++k) rest += (i128)r[k] * x[k];
            i64 b = ceil_div(to_i64(-rest), r[L]);
            lo = std::max(lo, b);
        }
        for (auto& r : s.upper[L]) {  // -|a| x_L + rest >= 0  ->  x_L <= floor(rest / |a|)
            i128 rest = r[d];
            for (int k = 0; k < L; ++k) rest += (i128)r[k] * x[k];
            i64 b = floor_div(to_i64(rest), -r[L]);
            up = std::min(up, b);
        }
    };
    int L = 0;
    i64 lo;
    bounds(0, lo, hi[0]);
    x[0] = lo;
    while (L >= 0) {
        if (x[L] > hi[L]) {
            --L;
            if (L >= 0) ++x[L];
            continue;
        }
        if (L == d - 1) {
            i64 n = hi[L] - x[L] + 1;
            budget_used += n;
            if (budget_used > max_points) throw PlanError{SP_ERR_UNSUPPORTED};
            for (; x[L] <= hi[L]; ++x[L]) f(x);
            continue;
        }
        ++L;
        bounds(L, lo, hi[L]);
        x[L] = lo;
    }
}

i64 exact_rank(std::vector<std::vector<i128>> A) {
    // fraction-free Gaussian elimination with gcd reduction of each row
    int rows = (int)A.size();
    if (rows == 0) return 0;
    int cols = (int)A[0].size();
    int r = 0;
    for (int c = 0; c < cols && r < rows; ++c) {
        int piv = -1;
        for (int i = r; i < rows; ++i)
            if (A[i][c] != 0) {
                piv = i;
                break;
            }
        if (piv < 0) continue;
        std::swap(A[r], A[piv]);
        for (int i = 0; i < rows; ++i) {
            if (i == r || A[i][c] == 0) continue;
            i128 a = A[r][c], b = A[i][c];
            i128 g = 0;
            for (int k = 0; k < cols; ++k) {
                A[i][k] = a * A[i][k] - b * A[r][k];
                i128 v = A[i][k] < 0 ? -A[i][k] : A[i][k];
                i128 x = g, y = v;
                while (y) {
                    i128 t = x % y;
                    x = y;
                    y = t;
                }
                g = x;
            }
            if (g > 1)
                for (int k = 0; k < cols; ++k) A[i][k] /= g;
        }
        ++r;
    }
    return r;
}

struct RefInfo {
    int stmt, array, is_write, rank, depth;
    std::vector<i64> F;   // rank x (depth + 1), parameters folded into the constant column
    bool nonempty = false;
    i64 lo[SP_MAX_RANK], hi[SP_MAX_RANK];
    std::vector<i64> keys;  // sorted unique linearised coordinates
};

i64 volume(const i64* lb, const i64* ub, int rank) {
    i128 v = 1;
    for (int k = 0; k < rank; ++k) {
        i128 e = (i128)ub[k] - lb[k] + 1;
        if (e <= 0) return 0;
        v *= e;
        if (v > (i128)INT64_MAX) throw PlanError{SP_ERR_OVERFLOW};
    }
    return (i64)v;
}

i64 intersect_count(const std::vector<i64>& a, const std::vector<i64>& b) {
    i64 n = 0;
    size_t i = 0, j = 0;
    while (i < a.size() && j < b.size()) {
        if (a[i] < b[j]) ++i;
        else if (b[j] < a[i]) ++j;
        else {
            ++n;
            ++i;
            ++j;
        }
    }
    return n;
}
bool intersects(const std::vector<i64>& a, const std::vector<i64>& b) {
    size_t i = 0, j = 0;
    while (i < a.size() && j < b.size()) {
        if (a[i] < b[j]) ++i;
        else if (b[j] < a[i]) ++j;
        else return true;
    }
    return false;
}

struct UF {
    std::vector<int> p;
    explicit UF(int n) : p(n) { std::iota(p.begin(), p.end(), 0); }
    int find(int x) {
        while (p[x] != x) x = p[x] = p[p[x]];
        return x;
    }
    void unite(int a, int b) { p[find(a)] = find(b); }
};

// connected components (overlap graph) among refs `ids`; each returned list sorted
std::vector<std::vector<int>> components(const std::vector<RefInfo>& R, const std::vector<int>& ids) {
    UF uf((int)ids.size());
    for (size_t i = 0; i < ids.size(); ++i)
        for (size_t j = i + 1; j < ids.size(); ++j)
            if (intersects(R[ids[i]].keys, R[ids[j]].keys)) uf.unite((int)i, (int)j);
    std::vector<std::vector<int>> groups;
    std::vector<int> gid(ids.size(), -1);
    for (size_t i = 0; i < ids.size(); ++i) {
        int root = uf.find((int)i);
        if (gid[root] < 0) {
            gid[root] = (int)groups.size();
            groups.push_back({});
        }
        groups[gid[root]].push_back(ids[i]);
    }
    return groups;  // ordered by smallest member since ids is ascending
}

void bbox_of(const std::vector<RefInfo>& R, const std::vector<int>& ids, int rank, i64* lb, i64* ub) {
    bool any = false;
    for (int k = 0; k < rank; ++k) {
        lb[k] = 0;
        ub[k] = -1;
    }
    for (int id : ids) {
        if (!R[id].nonempty) continue;
        for (int k = 0; k < rank; ++k) {
            if (!any || R[id].lo[k] < lb[k]) lb[k] = R[id].lo[k];
            if (!any || R[id].hi[k] > ub[k]) ub[k] = R[id].hi[k];
        }
        any = true;
    }
}

i64 union_count(const std::vector<RefInfo>& R, const std::vector<int>& ids) {
    std::vector<i64> all;
    for (int id : ids) all.insert(all.end(), R[id].keys.begin(), R[id].keys.end());
    std::sort(all.begin(), all.end());
    return (i64)(std::unique(all.begin(), all.end()) - all.begin());
}

// §3.1.2: the dimensions of the local array are those of the partition's
// convex hull; a global dimension that is an affine function of the earlier ones on the
// data spaces (CLooG scans dimensions in order and emits such a dimension as an expression,
// not a loop) is dropped.  On the affine hull p0 + span{p - p0}, dimension k is an affine
// function of dimensions 0..k-1 iff the projection of the span onto the first k+1
// coordinates has the same rank as onto the first k.  Those ranks are read off an echelon
// basis with leftmost-nonzero pivots (rank of the first k+1 columns = pivots <= k): the kept
// dimensions are exactly the pivot columns.  Exact integer arithmetic (gcd-normalised).
struct Echelon {
    int rank;
    int n = 0;
    i128 v[SP_MAX_RANK][SP_MAX_RANK];
    int piv[SP_MAX_RANK];
    explicit Echelon(int r) : rank(r) {}
    bool full() const { return n == rank; }
    void insert(const i64* d) {
        i128 x[SP_MAX_RANK];
        for (int k = 0; k < rank; ++k) x[k] = d[k];
        for (int b = 0; b < n; ++b) {  // basis kept sorted by pivot column
            const int c = piv[b];
            if (x[c] == 0) continue;
            const i128 xb = x[c], vb = v[b][c];
            i128 g = 0;
            for (int k = 0; k < rank; ++k) {
                x[k] = x[k] * vb - v[b][k] * xb;
                i128 a = x[k] < 0 ? -x[k] : x[k];
                for (i128 t = g; t != 0;) {  // g <- gcd(g, a)
                    const i128 r = a % t;
                    a = t;
                    t = r;
                }
                g = a;
            }
            if (g > 1)
                for (int k = 0; k < rank; ++k) x[k] /= g;
        }
        int c = 0;
        while (c < rank && x[c] == 0) ++c;
        if (c == rank) return;
        int pos = n;
        while (pos > 0 && piv[pos - 1] > c) {
            for (int k = 0; k < rank; ++k) v[pos][k] = v[pos - 1][k];
            piv[pos] = piv[pos - 1];
            --pos;
        }
        for (int k = 0; k < rank; ++k) v[pos][k] = x[k];
        piv[pos] = c;
        ++n;
    }
    int32_t mask() const {
        int32_t m = 0;
        for (int b = 0; b < n; ++b) m |= 1 << piv[b];
        return m;
    }
};

int plan_impl(const sp_block* blk, const sp_plan_opts* opts, sp_buffer* bufs, int32_t cap_bufs, int32_t* n_bufs,
              int32_t* ref_buf, int64_t* local_rows) {
    if (!blk || !n_bufs) return SP_ERR_INVALID_ARG;
    sp_plan_opts o{SP_PLAN_PER_ARRAY, 0, 0.30, 0, 0, 0, 0};
    if (opts) o = *opts;
    if (o.mode != SP_PLAN_PER_ARRAY && o.mode != SP_PLAN_COMPONENTS) return SP_ERR_INVALID_ARG;
    if ((o.compress != 0 && o.compress != 1) || o.reserved != 0) return SP_ERR_INVALID_ARG;
    if (o.mup_elems < 0 || o.max_points < 0 || !(o.delta >= 0.0)) return SP_ERR_INVALID_ARG;
    const i64 max_points = o.max_points ? o.max_points : kDefaultMaxPoints;
    const int P = blk->n_params, S = blk->n_stmts, NR = blk->n_refs;
    if (P < 0 || P > SP_MAX_PARAMS || S < 0 || NR < 0 || blk->reserved != 0) return SP_ERR_INVALID_ARG;
    if ((P > 0 && !blk->params) || (S > 0 && !blk->stmts) || (NR > 0 && !blk->refs)) return SP_ERR_INVALID_ARG;
    if (cap_bufs < 0 || (cap_bufs > 0 && !bufs)) return SP_ERR_INVALID_ARG;
    for (int s = 0; s < S; ++s) {
        const sp_domain& D = blk->stmts[s];
        if (D.depth < 0 || D.depth > SP_MAX_DEPTH || D.n_rows < 0 || (D.n_rows > 0 && !D.rows))
            return SP_ERR_INVALID_ARG;
    }
    for (int r = 0; r < NR; ++r) {
        const sp_ref& Rf = blk->refs[r];
        if (Rf.stmt < 0 || Rf.stmt >= S || Rf.rank < 1 || Rf.rank > SP_MAX_RANK || !Rf.rows)
            return SP_ERR_INVALID_ARG;
        for (int q = 0; q < r; ++q)
            if (blk->refs[q].array == Rf.array && blk->refs[q].rank != Rf.rank) return SP_ERR_INVALID_ARG;
    }

    // ---- statements: substitute parameters, build scanning bounds (CLooG role) ----
    std::vector<Scan> scans(S);
    for (int s = 0; s < S; ++s) {
        const sp_domain& D = blk->stmts[s];
        const int d = D.depth, W = d + P + 1;
        std::vector<Row> sys;
        for (int q = 0; q < D.n_rows; ++q) {
            const i64* row = D.rows + (size_t)q * W;
            Row r(d + 1);
            for (int k = 0; k < d; ++k) r[k] = row[k];
            i128 c = row[d + P];
            for (int p = 0; p < P; ++p) c += (i128)row[d + p] * blk->params[p];
            r[d] = to_i64(c);
            sys.push_back(r);
        }
        scans[s] = build_scan(sys, d);
    }

    // ---- references ----
    std::vector<RefInfo> R(NR);
    for (int r = 0; r < NR; ++r) {
        const sp_ref& Rf = blk->refs[r];
        RefInfo& I = R[r];
        I.stmt = Rf.stmt;
        I.array = Rf.array;
        I.is_write = Rf.is_write ? 1 : 0;
        I.rank = Rf.rank;
        I.depth = blk->stmts[Rf.stmt].depth;
        const int d = I.depth, W = d + P + 1;
        I.F.assign((size_t)I.rank * (d + 1), 0);
        for (int k = 0; k < I.rank; ++k) {
            const i64* row = Rf.rows + (size_t)k * W;
            for (int j = 0; j < d; ++j) I.F[k * (d + 1) + j] = row[j];
            i128 c = row[d + P];
            for (int p = 0; p < P; ++p) c += (i128)row[d + p] * blk->params[p];
            I.F[k * (d + 1) + d] = to_i64(c);
        }
    }
    auto image = [](const RefInfo& I, const i64* x, i64* out) {
        const int d = I.depth;
        for (int k = 0; k < I.rank; ++k) {
            const i64* f = &I.F[k * (d + 1)];
            i128 v = f[d];
            for (int j = 0; j < d; ++j) v += (i128)f[j] * x[j];
            out[k] = to_i64(v);
        }
    };

    // pass 1: exact per-ref bounding boxes of the data spaces (Alg. 2 step 3)
    i64 used = 0;
    for (int s = 0; s < S; ++s) {
        std::vector<int> mine;
        for (int r = 0; r < NR; ++r)
            if (R[r].stmt == s) mine.push_back(r);
        if (mine.empty()) continue;
        scan_points(scans[s], max_points, used, [&](const i64* x) {
            i64 c[SP_MAX_RANK];
            for (int r : mine) {
                RefInfo& I = R[r];
                image(I, x, c);
                for (int k = 0; k < I.rank; ++k) {
                    if (!I.nonempty || c[k] < I.lo[k]) I.lo[k] = c[k];
                    if (!I.nonempty || c[k] > I.hi[k]) I.hi[k] = c[k];
                }
                I.nonempty = true;
            }
        });
    }

    // per-array linearisation over the array's union bounding box
    std::vector<int> arrays;
    for (int r = 0; r < NR; ++r) arrays.push_back(R[r].array);
    std::sort(arrays.begin(), arrays.end());
    arrays.erase(std::unique(arrays.begin(), arrays.end()), arrays.end());
    struct Lin {
        int rank;
        i64 lo[SP_MAX_RANK], stride[SP_MAX_RANK];
    };
    std::vector<Lin> lin(arrays.size());
    std::vector<std::vector<int>> refs_of(arrays.size());
    for (size_t a = 0; a < arrays.size(); ++a) {
        for (int r = 0; r < NR; ++r)
            if (R[r].array == arrays[a]) refs_of[a].push_back(r);
        Lin& Ln = lin[a];
        Ln.rank = R[refs_of[a][0]].rank;
        i64 lb[SP_MAX_RANK], ub[SP_MAX_RANK];
        bbox_of(R, refs_of[a], Ln.rank, lb, ub);
        i128 st = 1;
        for (int k = Ln.rank - 1; k >= 0; --k) {
            Ln.lo[k] = lb[k];
            Ln.stride[k] = (i64)st;
            i128 e = (i128)ub[k] - lb[k] + 1;
            if (e < 1) e = 1;
            st *= e;
            if (st > ((i128)1 << 62)) throw PlanError{o.mode == SP_PLAN_PER_ARRAY ? SP_ERR_OVERFLOW : SP_ERR_UNSUPPORTED};
        }
    }
    std::vector<int> arr_index(NR);
    for (int r = 0; r < NR; ++r)
        arr_index[r] = (int)(std::lower_bound(arrays.begin(), arrays.end(), R[r].array) - arrays.begin());

    // pass 2: the data spaces themselves as sorted sets of linearised coordinates
    used = 0;
    for (int s = 0; s < S; ++s) {
        std::vector<int> mine;
        for (int r = 0; r < NR; ++r)
            if (R[r].stmt == s) mine.push_back(r);
        if (mine.empty()) continue;
        scan_points(scans[s], max_points, used, [&](const i64* x) {
            i64 c[SP_MAX_RANK];
            for (int r : mine) {
                RefInfo& I = R[r];
                image(I, x, c);
                const Lin& Ln = lin[arr_index[r]];
                i64 key = 0;
                for (int k = 0; k < I.rank; ++k) key += (c[k] - Ln.lo[k]) * Ln.stride[k];
                I.keys.push_back(key);
            }
        });
    }
    for (auto& I : R) {
        std::sort(I.keys.begin(), I.keys.end());
        I.keys.erase(std::unique(I.keys.begin(), I.keys.end()), I.keys.end());
    }

    // ---- partitions (Alg. 2 step 5) ----
    struct Part {
        int array_slot;
        std::vector<int> ids;
    };
    std::vector<Part> parts;
    for (size_t a = 0; a < arrays.size(); ++a) {
        if (o.mode == SP_PLAN_PER_ARRAY) parts.push_back({(int)a, refs_of[a]});
        else
            for (auto& g : components(R, refs_of[a])) parts.push_back({(int)a, g});
    }
    std::sort(parts.begin(), parts.end(), [&](const Part& x, const Part& y) {
        if (arrays[x.array_slot] != arrays[y.array_slot]) return arrays[x.array_slot] < arrays[y.array_slot];
        return x.ids.front() < y.ids.front();
    });

    std::vector<sp_buffer> out;
    std::vector<int32_t> rb(NR, -1);
    for (const Part& pt : parts) {
        sp_buffer b;
        std::memset(&b, 0, sizeof(b));
        const int rank = R[pt.ids[0]].rank;
        b.array = arrays[pt.array_slot];
        b.rank = rank;
        b.n_refs = (int32_t)pt.ids.size();
        bbox_of(R, pt.ids, rank, b.lb, b.ub);
        b.size = volume(b.lb, b.ub, rank);  // Alg. 2 step 9
        b.n_dims = rank;
        b.kept_mask = (int32_t)((1u << rank) - 1);
        if (o.compress) {  // §3.1.2: dimensions of the data spaces' affine hull only
            const Lin& Ln = lin[pt.array_slot];
            Echelon E(rank);
            bool have0 = false;
            i64 p0[SP_MAX_RANK], c[SP_MAX_RANK], dlt[SP_MAX_RANK];
            for (int id : pt.ids) {
                for (i64 key : R[id].keys) {
                    i64 rem = key;
                    for (int k = 0; k < rank; ++k) {
                        c[k] = Ln.lo[k] + rem / Ln.stride[k];
                        rem %= Ln.stride[k];
                    }
                    if (!have0) {
                        std::memcpy(p0, c, sizeof(i64) * rank);
                        have0 = true;
                        continue;
                    }
                    for (int k = 0; k < rank; ++k) dlt[k] = c[k] - p0[k];
                    E.insert(dlt);
                    if (E.full()) break;
                }
                if (E.full()) break;
            }
            b.n_dims = have0 ? E.n : 0;
            b.kept_mask = have0 ? E.mask() : 0;
            if (have0) {
                i128 sz = 1;
                for (int k = 0; k < rank; ++k)
                    if ((b.kept_mask >> k) & 1) sz *= (i128)b.ub[k] - b.lb[k] + 1;
                b.size = to_i64(sz);
            }
        }
        std::vector<int> rd, wr;
        for (int id : pt.ids) (R[id].is_write ? wr : rd).push_back(id);
        bbox_of(R, rd, rank, b.in_lb, b.in_ub);
        bbox_of(R, wr, rank, b.out_lb, b.out_ub);
        b.in_count = union_count(R, rd);
        b.out_count = union_count(R, wr);
        b.in_dense = b.in_count > 0 && b.in_count == volume(b.in_lb, b.in_ub, rank);
        b.out_dense = b.out_count > 0 && b.out_count == volume(b.out_lb, b.out_ub, rank);
        // upper bounds on moved volumes: components of read (write) spaces
        i128 vin = 0, vout = 0;
        for (auto& g : components(R, rd)) {
            i64 lb[SP_MAX_RANK], ub[SP_MAX_RANK];
            bbox_of(R, g, rank, lb, ub);
            vin += volume(lb, ub, rank);
        }
        for (auto& g : components(R, wr)) {
            i64 lb[SP_MAX_RANK], ub[SP_MAX_RANK];
            bbox_of(R, g, rank, lb, ub);
            vout += volume(lb, ub, rank);
        }
        b.v_in_ub = to_i64(vin);
        b.v_out_ub = to_i64(vout);
        // Algorithm 1: non-constant reuse (Cond. (1)), else constant reuse > delta
        b.union_count = union_count(R, pt.ids);
        i128 ov = 0;
        for (size_t i = 0; i < pt.ids.size(); ++i)
            for (size_t j = i + 1; j < pt.ids.size(); ++j) ov += intersect_count(R[pt.ids[i]].keys, R[pt.ids[j]].keys);
        b.overlap = to_i64(ov);
        bool ben = false;
        for (int id : pt.ids) {
            const RefInfo& I = R[id];
            std::vector<std::vector<i128>> M(I.rank, std::vector<i128>(I.depth));
            for (int k = 0; k < I.rank; ++k)
                for (int j = 0; j < I.depth; ++j) M[k][j] = I.F[k * (I.depth + 1) + j];
            if (I.depth > 0 && exact_rank(M) < I.depth) ben = true;
        }
        if (!ben && (double)b.overlap > o.delta * (double)b.union_count) ben = true;
        b.beneficial = ben ? 1 : 0;
        if (o.reuse_filter && !ben) continue;
        for (int id : pt.ids) rb[id] = (int32_t)out.size();
        out.push_back(b);
    }

    if ((i64)out.size() > cap_bufs) {
        *n_bufs = (int32_t)out.size();
        return SP_ERR_CAPACITY;
    }
    if (o.mup_elems > 0) {
        i128 tot = 0;
        for (auto& b : out) tot += b.size;
        if (tot > o.mup_elems) {
            *n_bufs = (int32_t)out.size();
            return SP_ERR_SMEM_LIMIT;
        }
    }
    // local access functions F' - g, in the caller's (i, p, 1) layout
    std::vector<i64> lr;
    for (int r = 0; r < NR; ++r) {
        const sp_ref& Rf = blk->refs[r];
        const int d = R[r].depth, W = d + P + 1;
        for (int k = 0; k < Rf.rank; ++k)
            for (int j = 0; j < W; ++j) {
                i64 v = Rf.rows[(size_t)k * W + j];
                if (j == W - 1 && rb[r] >= 0) v = to_i64((i128)v - out[rb[r]].lb[k]);
                if (rb[r] >= 0 && !((out[rb[r]].kept_mask >> k) & 1)) v = 0;  // F' drops the row
                lr.push_back(v);
            }
    }
    for (size_t i = 0; i < out.size(); ++i) bufs[i] = out[i];
    *n_bufs = (int32_t)out.size();
    if (ref_buf) std::memcpy(ref_buf, rb.data(), sizeof(int32_t) * NR);
    if (local_rows) std::memcpy(local_rows, lr.data(), sizeof(i64) * lr.size());
    return SP_OK;
}

}  // namespace

extern "C" int sp_plan_buffers(const sp_block* blk, const sp_plan_opts* opts, sp_buffer* bufs, int32_t cap_bufs,
                               int32_t* n_bufs, int32_t* ref_buf, int64_t* local_rows) {
    SP_NVTX("sp_plan_buffers");
    try {
        return plan_impl(blk, opts, bufs, cap_bufs, n_bufs, ref_buf, local_rows);
    } catch (const PlanError& e) {
        return e.code;
    } catch (...) {
        return SP_ERR_UNSUPPORTED;  // e.g. std::bad_alloc on an enormous block
    }
}

// ---------------------------------------------------------------------------------------
// Tile-size search (§4.3).
// For every candidate tile vector t the tile's iteration space is the box 0 <= i_l < t_l;
// Algorithm 2 (plan_impl, PER_ARRAY as in Figure 1) gives each array's local size M_k and
// move volumes V_in_k / V_out_k (§3.1.3).  Array k's movement code sits under the tiling
// loops 0..r_k, r_k = the deepest loop any of its references depends on (§4.2 hoisting), so
// it runs prod_{i<=r_k} ceil(N_i / t_i) times.  The paper relaxes t to reals and uses SQP
// (P:L788-794); here the objective is evaluated exactly on the caller's candidate grid.
// ---------------------------------------------------------------------------------------
namespace {

int tile_search_impl(const sp_tile_problem* pb, sp_tile_result* out) {
    if (!pb || !out) return SP_ERR_INVALID_ARG;
    const int m = pb->depth, nr = pb->n_refs;
    if (m < 1 || m > SP_MAX_DEPTH || nr < 1 || !pb->extent || !pb->refs || !pb->n_cand || !pb->cand || pb->procs < 1 ||
        pb->mup_elems < 0 || pb->reserved != 0)
        return SP_ERR_INVALID_ARG;
    std::vector<std::vector<i64>> cand(m);
    size_t off = 0;
    for (int l = 0; l < m; ++l) {
        if (pb->n_cand[l] < 1 || pb->extent[l] < 1) return SP_ERR_INVALID_ARG;
        for (int q = 0; q < pb->n_cand[l]; ++q) {
            const i64 t = pb->cand[off + q];
            if (t < 1 || t > pb->extent[l]) return SP_ERR_INVALID_ARG;  // 0 < t_i <= N_i
            cand[l].push_back(t);
        }
        off += pb->n_cand[l];
    }
    // r_k per array id: deepest loop with a nonzero coefficient in any of its refs
    std::vector<int> arrays;
    for (int r = 0; r < nr; ++r) arrays.push_back(pb->refs[r].array);
    std::sort(arrays.begin(), arrays.end());
    arrays.erase(std::unique(arrays.begin(), arrays.end()), arrays.end());
    std::vector<int> rk(arrays.size(), -1);
    for (int r = 0; r < nr; ++r) {
        const sp_ref& R = pb->refs[r];
        if (R.rank < 1 || R.rank > SP_MAX_RANK || !R.rows) return SP_ERR_INVALID_ARG;
        const size_t a = std::lower_bound(arrays.begin(), arrays.end(), R.array) - arrays.begin();
        for (int k = 0; k < R.rank; ++k)
            for (int l = 0; l < m; ++l)
                if (R.rows[(size_t)k * (m + 1) + l] != 0 && l > rk[a]) rk[a] = l;
    }
    std::vector<sp_ref> refs(pb->refs, pb->refs + nr);
    for (auto& R : refs) R.stmt = 0;
    std::vector<i64> rows(2 * (size_t)m * (m + 1), 0);
    sp_domain dom{m, 2 * m, rows.data()};
    sp_block blk{0, 1, nr, 0, nullptr, &dom, refs.data()};
    sp_plan_opts opts{SP_PLAN_PER_ARRAY, 0, 0.30, 0, 0};
    std::vector<sp_buffer> bufs(arrays.size());
    std::vector<size_t> idx(m, 0);
    std::memset(out, 0, sizeof(*out));
    out->cost = 0.0;
    bool have = false;
    i64 evaluated = 0;
    for (;;) {
        i64 t[SP_MAX_DEPTH];
        i128 prod = 1;
        for (int l = 0; l < m; ++l) {
            t[l] = cand[l][idx[l]];
            prod *= t[l];
        }
        if (prod >= pb->procs) {  // t_1 x ... x t_m >= P
            for (int l = 0; l < m; ++l) {  // box 0 <= i_l <= t_l - 1
                i64* r0 = &rows[(size_t)(2 * l) * (m + 1)];
                i64* r1 = &rows[(size_t)(2 * l + 1) * (m + 1)];
                std::fill(r0, r0 + m + 1, 0);
                std::fill(r1, r1 + m + 1, 0);
                r0[l] = 1;
                r1[l] = -1;
                r1[m] = t[l] - 1;
            }
            int32_t nb = 0;
            const int st = plan_impl(&blk, &opts, bufs.data(), (int32_t)bufs.size(), &nb, nullptr, nullptr);
            if (st) return st;
            ++evaluated;
            i128 mem = 0;
            double cost = 0.0;
            for (int b = 0; b < nb; ++b) {
                mem += bufs[b].size;
                const size_t a = std::lower_bound(arrays.begin(), arrays.end(), bufs[b].array) - arrays.begin();
                double moves = 1.0;
                for (int l = 0; l <= rk[a]; ++l) moves *= (double)((pb->extent[l] + t[l] - 1) / t[l]);
                const double P = (double)pb->procs;
                if (bufs[b].in_count > 0) cost += moves * (P * pb->sync_cost + (double)bufs[b].v_in_ub * pb->elem_cost / P);
                if (bufs[b].out_count > 0)
                    cost += moves * (P * pb->sync_cost + (double)bufs[b].v_out_ub * pb->elem_cost / P);
            }
            if ((pb->mup_elems == 0 || mem <= pb->mup_elems) && (!have || cost < out->cost)) {
                have = true;
                out->cost = cost;
                out->local_elems = (i64)mem;
                for (int l = 0; l < m; ++l) out->tile[l] = t[l];
            }
        }
        int l = m - 1;
        while (l >= 0 && ++idx[l] == cand[l].size()) idx[l--] = 0;
        if (l < 0) break;
    }
    out->evaluated = evaluated;
    out->feasible = have ? 1 : 0;
    return SP_OK;
}

}  // namespace

extern "C" int sp_tile_search(const sp_tile_problem* prob, sp_tile_result* out) {
    SP_NVTX("sp_tile_search");
    try {
        return tile_search_impl(prob, out);
    } catch (const PlanError& e) {
        return e.code;
    } catch (...) {
        return SP_ERR_UNSUPPORTED;
    }
}

// ---------------------------------------------------------------------------------------
// Domain enumeration for the staged-tile executor (exec.cu): the integer points of one
// statement polytope with concrete parameters, in lexicographic loop order.
// ---------------------------------------------------------------------------------------
namespace sp {
int enumerate_domain(const sp_domain& D, int n_params, const int64_t* params, int64_t max_points,
                     std::vector<int64_t>& out, int64_t* count) {
    try {
        const int d = D.depth, W = d + n_params + 1;
        if (d < 0 || d > SP_MAX_DEPTH || D.n_rows < 0 || (D.n_rows > 0 && !D.rows)) return SP_ERR_INVALID_ARG;
        std::vector<Row> sys;
        for (int q = 0; q < D.n_rows; ++q) {
            const i64* row = D.rows + (size_t)q * W;
            Row r(d + 1);
            for (int k = 0; k < d; ++k) r[k] = row[k];
            i128 c = row[d + n_params];
            for (int p = 0; p < n_params; ++p) c += (i128)row[d + p] * params[p];
            r[d] = to_i64(c);
            sys.push_back(r);
        }
        const Scan sc = build_scan(sys, d);
        i64 used = 0;
        i64 n = 0;
        scan_points(sc, max_points > 0 ? max_points : kDefaultMaxPoints, used, [&](const i64* x) {
            out.insert(out.end(), x, x + d);
            ++n;
        });
        *count = n;
        return SP_OK;
    } catch (const PlanError& e) {
        return e.code;
    } catch (...) {
        return SP_ERR_UNSUPPORTED;
    }
}
}  // namespace sp

// exec.cu — generic staged-tile executor: an arbitrary small affine
// program block runs on the GPU the way the paper's framework prescribes (sp.h section 6).
//
// Host ("compiler", once per call):
//   for every tile (the block with that tile's parameter values)
//     * sp_plan_buffers (PER_ARRAY: one bounding box per array, Figure 1 / Alg. 2) gives
//       the local buffers, which references are staged, and the local access functions
//       F'(y) - g;
//     * the statement instances are enumerated and put in original program order (the
//       2d+1 schedule of each body's textual positions);
//     * each instance's operands become addresses: shared-memory index through F' - g
//       for staged references, global index through F otherwise;
//     * move-in = every element of the union of the read data spaces of a buffer, move-out
//       = every element of the union of its write data spaces;
//     * instances are grouped into dependence levels: an instance's level is one more than
//       that of the latest earlier instance it conflicts with (flow, anti or output
//       dependence on one element), so a level's instances are independent.
//   Consecutive tiles of one CTA keep a buffer resident when its read and write data
//   spaces are the same in both (§4.2 hoisting: the tiling loop is redundant for it).
// Device (one CTA per group of tiles): segments of moves and levels, __syncthreads between
// segments; each thread evaluates its instances' postfix bodies in fp32 (explicit _rn ops).
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <exception>
#include <map>
#include <unordered_map>
#include <vector>

#include "../../include/sp.h"
#include "sp_internal.h"

namespace {

constexpr int kStack = 16;
constexpr int kThreads = 256;
enum { kSegIn = 0, kSegExec = 1, kSegOut = 2 };

struct ExecArgs {
    const int32_t* runs;   // [ctas][2]: first segment, segment count
    const int32_t* segs;   // [n][3]: kind, first item, item count
    const int32_t* moves;  // [n][3]: array, global index, shared index
    const int32_t* insts;  // [n][rec]: stmt, (array, index) of the write, (array, index) per LOAD
    const int32_t* code;   // [n][2]: op, arg (LOAD: operand slot, CONST: float bits)
    const int32_t* stmt_code;  // [stmts][2]: first instruction, count
    float* const* arrays;  // [n_arrays]
    int32_t rec;
};

__device__ __forceinline__ float* operand(const ExecArgs& a, float* sm, int32_t arr, int32_t idx) {
    return arr < 0 ? sm + idx : a.arrays[arr] + idx;
}

__global__ void __launch_bounds__(kThreads) exec_kernel(ExecArgs a) {
    extern __shared__ float sm[];
    const int32_t seg0 = a.runs[2 * blockIdx.x], nseg = a.runs[2 * blockIdx.x + 1];
    for (int q = 0; q < nseg; ++q) {
        const int32_t* sg = a.segs + 3 * (seg0 + q);
        const int kind = sg[0], first = sg[1], count = sg[2];
        if (kind == kSegExec) {
            for (int i = threadIdx.x; i < count; i += blockDim.x) {
                const int32_t* r = a.insts + (size_t)(first + i) * a.rec;
                const int32_t* c = a.code + 2 * a.stmt_code[2 * r[0]];
                const int n = a.stmt_code[2 * r[0] + 1];
                float st[kStack];
                int sp = 0;
                for (int k = 0; k < n; ++k) {
                    const int op = c[2 * k], arg = c[2 * k + 1];
                    if (op == SP_OP_LOAD) {
                        st[sp++] = *operand(a, sm, r[3 + 2 * arg], r[4 + 2 * arg]);
                    } else if (op == SP_OP_CONST) {
                        st[sp++] = __int_as_float(arg);
                    } else {
                        const float y = st[--sp], x = st[sp - 1];
                        st[sp - 1] = op == SP_OP_ADD ? __fadd_rn(x, y) : op == SP_OP_SUB ? __fsub_rn(x, y) : __fmul_rn(x, y);
                    }
                }
                *operand(a, sm, r[1], r[2]) = st[0];
            }
        } else {
            for (int i = threadIdx.x; i < count; i += blockDim.x) {
                const int32_t* m = a.moves + 3 * (size_t)(first + i);
                if (kind == kSegIn) sm[m[2]] = a.arrays[m[0]][m[1]];
                else a.arrays[m[0]][m[1]] = sm[m[2]];
            }
        }
        __syncthreads();
    }
}

struct Error {
    int code;
};

// ---- per-tile compilation -------------------------------------------------------------
struct Inst {
    std::vector<int64_t> key;      // 2d+1 schedule key (original order)
    std::vector<int32_t> rec;      // device record
    int64_t w_elem;                // element keys: array << 40 | global flat index
    std::vector<int64_t> r_elems;
    int level;
};

struct TileInfo {
    std::vector<sp_buffer> bufs;          // planner output
    std::vector<int32_t> ref_buf;         // per ref
    std::vector<int64_t> local_rows;      // per ref, rank x (depth + P + 1)
    std::vector<std::vector<int64_t>> rd, wr;  // per array id: sorted element keys read / written via staged refs
    std::vector<Inst> list;                    // instances in original program order
    std::vector<std::vector<int64_t>> din, dout;  // SP_MOVE_DATAFLOW: the §3.1.4 subsets of rd / wr
};

struct Group {  // the tiles one CTA runs, and its shared-memory slot per array
    std::vector<TileInfo> tiles;
    std::vector<int64_t> slot_off;
};

int64_t dot(const int64_t* row, const int64_t* x, int d, const int64_t* p, int P) {
    __int128 v = row[d + P];
    for (int k = 0; k < d; ++k) v += (__int128)row[k] * x[k];
    for (int k = 0; k < P; ++k) v += (__int128)row[d + k] * p[k];
    if (v > INT64_MAX || v < INT64_MIN) throw Error{SP_ERR_OVERFLOW};
    return (int64_t)v;
}

struct Compiler {
    const sp_block& blk;
    const sp_stmt_body* bodies;
    const sp_array_desc* arrays;
    int n_arrays;
    sp_exec_opts o;
    // outputs
    std::vector<int32_t> runs, segs, moves, insts, code, stmt_code;
    std::vector<Group> groups;
    int rec = 3;
    int32_t smem_elems = 0;
    sp_exec_stats st{};

    int64_t global_index(int arr, const int64_t* c) const {
        const sp_array_desc& A = arrays[arr];
        int64_t idx = 0;
        for (int k = 0; k < A.rank; ++k) {
            if (c[k] < 0 || c[k] >= A.extent[k]) throw Error{SP_ERR_INVALID_ARG};
            idx = idx * A.extent[k] + c[k];
        }
        if (idx > INT32_MAX) throw Error{SP_ERR_UNSUPPORTED};
        return idx;
    }

    TileInfo plan(const int64_t* params) const {
        sp_block b = blk;
        b.params = params;
        sp_plan_opts po{SP_PLAN_PER_ARRAY, o.reuse_filter, 0.30, 0, o.max_points, o.compress, 0};
        TileInfo t;
        int32_t nb = 0;
        t.bufs.resize(std::max(1, n_arrays));
        t.ref_buf.resize(std::max(1, blk.n_refs));
        size_t width = 0;
        for (int r = 0; r < blk.n_refs; ++r)
            width += (size_t)blk.refs[r].rank * (blk.stmts[blk.refs[r].stmt].depth + blk.n_params + 1);
        t.local_rows.resize(std::max<size_t>(1, width));
        int s = sp_plan_buffers(&b, &po, t.bufs.data(), (int32_t)t.bufs.size(), &nb, t.ref_buf.data(), t.local_rows.data());
        if (s) throw Error{s};
        t.bufs.resize(nb);
        t.rd.assign(n_arrays, {});
        t.wr.assign(n_arrays, {});
        return t;
    }

    bool live_out(int64_t e) const { return !o.live_out || o.live_out[e >> 40]; }

    // §3.1.4, exact on instances, with the tiles in order as the program:
    //   move in  = elements a tile reads before writing them itself (their value comes from
    //              an earlier tile or from the input),
    //   move out = elements whose last write in the tile is read by a later tile before it
    //              is rewritten, or that no later tile rewrites while their array is live-out.
    void dataflow() {
        std::vector<TileInfo*> all;
        for (Group& g : groups)
            for (TileInfo& t : g.tiles) all.push_back(&t);
        std::vector<std::unordered_map<int64_t, char>> exposed(all.size()), written(all.size());
        for (size_t t = 0; t < all.size(); ++t) {
            auto& W = written[t];
            for (const Inst& I : all[t]->list) {
                for (int64_t e : I.r_elems)
                    if (!W.count(e)) exposed[t][e] = 1;
                W[I.w_elem] = 1;
            }
        }
        std::unordered_map<int64_t, char> needed;  // after tile t: is the value of e needed later?
        for (size_t t = all.size(); t-- > 0;) {
            TileInfo& T = *all[t];
            T.din.assign(n_arrays, {});
            T.dout.assign(n_arrays, {});
            for (int a = 0; a < n_arrays; ++a) {
                for (int64_t e : T.wr[a]) {
                    auto it = needed.find(e);
                    if (it != needed.end() ? it->second : live_out(e)) T.dout[a].push_back(e);
                }
                for (int64_t e : T.rd[a])
                    if (exposed[t].count(e)) T.din[a].push_back(e);
            }
            for (auto& kv : written[t]) needed[kv.first] = 0;
            for (auto& kv : exposed[t]) needed[kv.first] = 1;
        }
    }

    void compile() {
        const int P = blk.n_params, S = blk.n_stmts, NR = blk.n_refs;
        // statement code table
        int max_loads = 0;
        stmt_code.resize(2 * S);
        for (int s = 0; s < S; ++s) {
            const sp_stmt_body& B = bodies[s];
            stmt_code[2 * s] = (int32_t)(code.size() / 2);
            stmt_code[2 * s + 1] = B.n_ops;
            int loads = 0, depth = 0;
            if (B.n_ops < 1 || !B.ops || !B.beta || B.write_ref < 0 || B.write_ref >= NR) throw Error{SP_ERR_INVALID_ARG};
            const sp_ref& W = blk.refs[B.write_ref];
            if (W.stmt != s || !W.is_write) throw Error{SP_ERR_INVALID_ARG};
            for (int k = 0; k < B.n_ops; ++k) {
                const sp_op& op = B.ops[k];
                int32_t arg = 0;
                if (op.op == SP_OP_LOAD) {
                    if (op.ref < 0 || op.ref >= NR || blk.refs[op.ref].stmt != s || blk.refs[op.ref].is_write)
                        throw Error{SP_ERR_INVALID_ARG};
                    arg = loads++;
                    ++depth;
                } else if (op.op == SP_OP_CONST) {
                    std::memcpy(&arg, &op.value, 4);
                    ++depth;
                } else if (op.op == SP_OP_ADD || op.op == SP_OP_SUB || op.op == SP_OP_MUL) {
                    if (depth < 2) throw Error{SP_ERR_INVALID_ARG};
                    --depth;
                } else {
                    throw Error{SP_ERR_INVALID_ARG};
                }
                if (depth > kStack) throw Error{SP_ERR_UNSUPPORTED};
                code.push_back(op.op);
                code.push_back(arg);
            }
            if (depth != 1) throw Error{SP_ERR_INVALID_ARG};
            max_loads = std::max(max_loads, loads);
        }
        rec = 3 + 2 * max_loads;
        for (int r = 0; r < NR; ++r) {
            const sp_ref& R = blk.refs[r];
            if (R.array < 0 || R.array >= n_arrays || arrays[R.array].rank != R.rank || !arrays[R.array].data)
                throw Error{SP_ERR_INVALID_ARG};
        }

        const int T = o.n_tiles, G = o.tiles_per_cta;
        const int64_t* tp = o.tile_params ? o.tile_params : blk.params;
        for (int g0 = 0; g0 < T; g0 += G) {
            const int g1 = std::min(T, g0 + G);
            std::vector<TileInfo> tiles;
            for (int t = g0; t < g1; ++t) tiles.push_back(plan(tp + (size_t)t * P));
            // shared-memory slot per array: the largest buffer of the group
            std::vector<int64_t> slot_size(n_arrays, 0), slot_off(n_arrays, 0);
            for (auto& ti : tiles)
                for (auto& b : ti.bufs) slot_size[b.array] = std::max(slot_size[b.array], b.size);
            int64_t tot = 0;
            for (int a = 0; a < n_arrays; ++a) {
                slot_off[a] = tot;
                tot += slot_size[a];
            }
            if (tot * 4 > 227 * 1024) throw Error{SP_ERR_SMEM_LIMIT};
            smem_elems = std::max<int32_t>(smem_elems, (int32_t)tot);

            // instances, operands, data spaces, levels — per tile
            for (size_t ti = 0; ti < tiles.size(); ++ti) {
                TileInfo& TI = tiles[ti];
                const int64_t* params = tp + (size_t)(g0 + ti) * P;
                // buffer of each array (PER_ARRAY: at most one)
                std::vector<int> buf_of(n_arrays, -1);
                for (size_t b = 0; b < TI.bufs.size(); ++b) buf_of[TI.bufs[b].array] = (int)b;
                size_t lr_pos = 0;
                std::vector<size_t> lr_at(NR);
                for (int r = 0; r < NR; ++r) {
                    lr_at[r] = lr_pos;
                    lr_pos += (size_t)blk.refs[r].rank * (blk.stmts[blk.refs[r].stmt].depth + P + 1);
                }
                std::vector<Inst>& list = TI.list;
                for (int s = 0; s < S; ++s) {
                    const sp_domain& D = blk.stmts[s];
                    const int d = D.depth;
                    std::vector<int64_t> pts;
                    int64_t count = 0;
                    const int e = sp::enumerate_domain(D, P, params, o.max_points, pts, &count);
                    if (e) throw Error{e};
                    const sp_stmt_body& B = bodies[s];
                    std::vector<int> loads;
                    for (int k = 0; k < B.n_ops; ++k)
                        if (B.ops[k].op == SP_OP_LOAD) loads.push_back(B.ops[k].ref);
                    for (int64_t q = 0; q < count; ++q) {
                        const int64_t* x = d ? &pts[q * d] : nullptr;
                        Inst I;
                        I.key.reserve(2 * d + 1);
                        for (int k = 0; k < d; ++k) {
                            I.key.push_back(B.beta[k]);
                            I.key.push_back(x[k]);
                        }
                        I.key.push_back(B.beta[d]);
                        I.rec.assign(rec, 0);
                        I.rec[0] = s;
                        auto addr = [&](int r, int32_t* out2, int64_t* elem) {
                            const sp_ref& R = blk.refs[r];
                            int64_t c[SP_MAX_RANK];
                            for (int k = 0; k < R.rank; ++k) c[k] = dot(R.rows + (size_t)k * (d + P + 1), x, d, params, P);
                            const int64_t gi = global_index(R.array, c);
                            *elem = (int64_t)R.array << 40 | gi;
                            const int b = TI.ref_buf[r];
                            if (b < 0) {
                                out2[0] = R.array;
                                out2[1] = (int32_t)gi;
                                return false;
                            }
                            // local access function F' - g (planner output) -> local coordinates
                            const sp_buffer& Bf = TI.bufs[b];
                            int64_t li = 0;
                            for (int k = 0; k < R.rank; ++k) {
                                const int64_t lc = dot(&TI.local_rows[lr_at[r] + (size_t)k * (d + P + 1)], x, d, params, P);
                                const int64_t ext = ((Bf.kept_mask >> k) & 1) ? Bf.ub[k] - Bf.lb[k] + 1 : 1;
                                if (lc < 0 || lc >= ext) throw Error{SP_ERR_UNSUPPORTED};  // planner invariant
                                li = li * ext + lc;
                            }
                            out2[0] = -1;
                            out2[1] = (int32_t)(slot_off[R.array] + li);
                            return true;
                        };
                        int64_t we;
                        if (addr(B.write_ref, &I.rec[1], &we)) TI.wr[blk.refs[B.write_ref].array].push_back(we);
                        I.w_elem = we;
                        for (size_t l = 0; l < loads.size(); ++l) {
                            int64_t re;
                            if (addr(loads[l], &I.rec[3 + 2 * l], &re)) TI.rd[blk.refs[loads[l]].array].push_back(re);
                            I.r_elems.push_back(re);
                        }
                        list.push_back(std::move(I));
                    }
                }
                std::stable_sort(list.begin(), list.end(), [](const Inst& a, const Inst& b) { return a.key < b.key; });
                // dependence levels (exact, per element, in program order)
                std::unordered_map<int64_t, int> lw, lr;
                for (Inst& I : list) {
                    int lv = 0;
                    for (int64_t e : I.r_elems) {
                        auto it = lw.find(e);
                        if (it != lw.end()) lv = std::max(lv, it->second + 1);
                    }
                    {
                        auto it = lw.find(I.w_elem);
                        if (it != lw.end()) lv = std::max(lv, it->second + 1);
                        auto jt = lr.find(I.w_elem);
                        if (jt != lr.end()) lv = std::max(lv, jt->second + 1);
                    }
                    I.level = lv;
                    for (int64_t e : I.r_elems) {
                        int& v = lr[e];
                        v = std::max(v, lv);
                    }
                    lw[I.w_elem] = lv;
                }
                for (int a = 0; a < n_arrays; ++a) {
                    for (auto* v : {&TI.rd[a], &TI.wr[a]}) {
                        std::sort(v->begin(), v->end());
                        v->erase(std::unique(v->begin(), v->end()), v->end());
                    }
                }
            }

            groups.push_back(Group{std::move(tiles), std::move(slot_off)});
        }
        if (o.movement == SP_MOVE_DATAFLOW) dataflow();
        int64_t tile_base = 0;
        for (Group& grp : groups) {
            std::vector<TileInfo>& tiles = grp.tiles;
            const std::vector<int64_t>& slot_off = grp.slot_off;
            // emit the CTA's segments
            const int32_t seg_first = (int32_t)(segs.size() / 3);
            auto emit_moves = [&](int kind, const TileInfo& TI, int a, int64_t tile) {
                const bool df = o.movement == SP_MOVE_DATAFLOW;
                const std::vector<int64_t>& set = kind == kSegIn ? (df ? TI.din[a] : TI.rd[a]) : (df ? TI.dout[a] : TI.wr[a]);
                if (o.move_counts) o.move_counts[(tile * n_arrays + a) * 2 + (kind == kSegIn ? 0 : 1)] = (int64_t)set.size();
                if (set.empty()) return;
                const sp_buffer* Bf = nullptr;
                for (auto& b : TI.bufs)
                    if (b.array == a) Bf = &b;
                const int32_t first = (int32_t)(moves.size() / 3);
                const sp_array_desc& A = arrays[a];
                for (int64_t e : set) {
                    const int64_t gi = e & ((int64_t(1) << 40) - 1);
                    // global coordinates -> local index in the buffer's bounding box
                    int64_t c[SP_MAX_RANK], rem = gi;
                    for (int k = A.rank - 1; k >= 0; --k) {
                        c[k] = rem % A.extent[k];
                        rem /= A.extent[k];
                    }
                    int64_t li = 0;
                    for (int k = 0; k < A.rank; ++k)  // dropped dimensions (§3.1.2): extent 1, index 0
                        if ((Bf->kept_mask >> k) & 1) li = li * (Bf->ub[k] - Bf->lb[k] + 1) + (c[k] - Bf->lb[k]);
                    moves.push_back(a);
                    moves.push_back((int32_t)gi);
                    moves.push_back((int32_t)(slot_off[a] + li));
                }
                const int32_t n = (int32_t)(moves.size() / 3) - first;
                if (kind == kSegIn) st.moved_in += n;
                else st.moved_out += n;
                segs.push_back(kind);
                segs.push_back(first);
                segs.push_back(n);
            };
            auto same_spaces = [&](const TileInfo& x, const TileInfo& y, int a) {
                return x.rd[a] == y.rd[a] && x.wr[a] == y.wr[a];
            };
            const bool hoist = o.hoist && o.movement != SP_MOVE_DATAFLOW;
            for (size_t ti = 0; ti < tiles.size(); ++ti) {
                const TileInfo& TI = tiles[ti];
                const int64_t tile = tile_base + (int64_t)ti;
                for (int a = 0; a < n_arrays; ++a) {
                    const bool resident = hoist && ti > 0 && same_spaces(tiles[ti - 1], TI, a);
                    if (resident) {
                        st.moves_hoisted += (int64_t)TI.rd[a].size();
                        if (o.move_counts) o.move_counts[(tile * n_arrays + a) * 2] = 0;
                    } else {
                        emit_moves(kSegIn, TI, a, tile);
                    }
                }
                std::vector<Inst>& list = tiles[ti].list;
                int nl = 0;
                for (auto& I : list) nl = std::max(nl, I.level + 1);
                st.max_levels = std::max(st.max_levels, nl);
                st.instances += (int64_t)list.size();
                std::stable_sort(list.begin(), list.end(), [](const Inst& a, const Inst& b) { return a.level < b.level; });
                size_t q = 0;
                for (int lv = 0; lv < nl; ++lv) {
                    const int32_t first = (int32_t)(insts.size() / rec);
                    for (; q < list.size() && list[q].level == lv; ++q)
                        insts.insert(insts.end(), list[q].rec.begin(), list[q].rec.end());
                    segs.push_back(kSegExec);
                    segs.push_back(first);
                    segs.push_back((int32_t)(insts.size() / rec) - first);
                }
                for (int a = 0; a < n_arrays; ++a) {
                    const bool stays = hoist && ti + 1 < tiles.size() && same_spaces(tiles[ti + 1], TI, a);
                    if (stays) {
                        st.moves_hoisted += (int64_t)TI.wr[a].size();
                        if (o.move_counts) o.move_counts[(tile * n_arrays + a) * 2 + 1] = 0;
                    } else {
                        emit_moves(kSegOut, TI, a, tile);
                    }
                }
            }
            tile_base += (int64_t)tiles.size();
            runs.push_back(seg_first);
            runs.push_back((int32_t)(segs.size() / 3) - seg_first);
        }
        st.ctas = (int32_t)(runs.size() / 2);
        st.smem_bytes = smem_elems * 4;
    }
};

template <class T>
int upload(const std::vector<T>& v, void** dev, cudaStream_t s) {
    const size_t bytes = std::max<size_t>(sizeof(T), v.size() * sizeof(T));
    SP_CUDA_TRY(cudaMallocAsync(dev, bytes, s));
    if (!v.empty()) SP_CUDA_TRY(cudaMemcpyAsync(*dev, v.data(), v.size() * sizeof(T), cudaMemcpyHostToDevice, s));
    return SP_OK;
}

}  // namespace

extern "C" int sp_exec_block(const sp_block* blk, const sp_stmt_body* bodies, const sp_array_desc* arrays,
                             int32_t n_arrays, const sp_exec_opts* opts, sp_exec_stats* stats, void* stream) {
    SP_NVTX("sp_exec_block");
    if (!blk || !bodies || !arrays || n_arrays < 1 || !opts) return SP_ERR_INVALID_ARG;
    if (opts->n_tiles < 1 || opts->tiles_per_cta < 1) return SP_ERR_INVALID_ARG;
    if (opts->movement != SP_MOVE_ALL && opts->movement != SP_MOVE_DATAFLOW) return SP_ERR_INVALID_ARG;
    if ((opts->compress != 0 && opts->compress != 1) || opts->reserved != 0) return SP_ERR_INVALID_ARG;
    if (blk->n_params > 0 && !opts->tile_params && !(opts->n_tiles == 1 && blk->params)) return SP_ERR_INVALID_ARG;
    for (int a = 0; a < n_arrays; ++a)
        if (arrays[a].rank < 1 || arrays[a].rank > SP_MAX_RANK) return SP_ERR_INVALID_ARG;
    Compiler C{*blk, bodies, arrays, n_arrays, *opts};
    try {
        C.compile();
    } catch (const Error& e) {
        return e.code;
    } catch (const std::exception& e) {
        if (getenv("SP_EXEC_DEBUG")) fprintf(stderr, "sp_exec_block: %s\n", e.what());
        return SP_ERR_UNSUPPORTED;
    }
    if (stats) *stats = C.st;
    if (opts->dry_run) return SP_OK;
    const cudaStream_t s = (cudaStream_t)stream;
    std::vector<float*> ptrs(n_arrays);
    for (int a = 0; a < n_arrays; ++a) ptrs[a] = arrays[a].data;
    void *d_runs = nullptr, *d_segs = nullptr, *d_moves = nullptr, *d_insts = nullptr, *d_code = nullptr,
         *d_sc = nullptr, *d_ptrs = nullptr;
    int st = SP_OK;
    if (!st) st = upload(C.runs, &d_runs, s);
    if (!st) st = upload(C.segs, &d_segs, s);
    if (!st) st = upload(C.moves, &d_moves, s);
    if (!st) st = upload(C.insts, &d_insts, s);
    if (!st) st = upload(C.code, &d_code, s);
    if (!st) st = upload(C.stmt_code, &d_sc, s);
    if (!st) st = upload(ptrs, &d_ptrs, s);
    if (!st) {
        ExecArgs a{(const int32_t*)d_runs, (const int32_t*)d_segs, (const int32_t*)d_moves, (const int32_t*)d_insts,
                   (const int32_t*)d_code, (const int32_t*)d_sc, (float* const*)d_ptrs, C.rec};
        const int smem = C.smem_elems * 4;
        cudaError_t e = cudaFuncSetAttribute(exec_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
        if (e == cudaSuccess) {
            exec_kernel<<<C.st.ctas, kThreads, smem, s>>>(a);
            e = cudaGetLastError();
        }
        if (e != cudaSuccess) {
            sp::set_cuda_error((int)e);
            st = SP_ERR_CUDA;
        }
    }
    // the host vectors were copied by cudaMemcpyAsync from pageable memory (staged before
    // return); the device copies are freed in stream order after the kernel
    for (void* p : {d_runs, d_segs, d_moves, d_insts, d_code, d_sc, d_ptrs})
        if (p) cudaFreeAsync(p, s);
    return st;
}

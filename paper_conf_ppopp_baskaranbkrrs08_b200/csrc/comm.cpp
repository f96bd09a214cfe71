// comm.cpp — multi-GPU layer: one process per GPU, NCCL over NVLink.
//
// Jacobi is partitioned into contiguous slabs; before each time tile (pass) the ranks
// exchange H = halo(Tt) boundary cells with each neighbour, then every rank runs the
// segment pass kernel (jacobi.cu) on [x_begin - H, x_end + H).  This is the only exchange
// step of the path (the paper's single-GPU "synchronization across all thread blocks",
// P:L861-862, becomes a kernel boundary plus a neighbour exchange across GPUs).
// ME needs no exchange during the search (independent macroblocks); results are gathered
// with ncclAllGather.
//
// NCCL is loaded at run time (dlopen of libnccl.so.2, or $SP_NCCL_LIB) so libsp has no
// link-time dependency on it.  The same pass loop also drives a single-GPU "loopback"
// transport (virtual ranks on one device, halos moved by cudaMemcpyAsync), which lets the
// partitioned path be tested on a one-GPU box.
#include <cuda_runtime.h>
#include <dlfcn.h>

#include <chrono>
#include <cstdlib>
#include <thread>
#include <cstring>
#include <mutex>
#include <vector>

#include "../../include/sp.h"
#include "sp_internal.h"
#include "sp_nccl_min.h"

struct sp_comm {
    ncclComm_t comm = nullptr;
    int32_t rank = 0, nranks = 1, device = 0;
    cudaStream_t side = nullptr;     // halo exchange of the overlapped pass loop
    cudaEvent_t ev_edge = nullptr;   // edge tiles of a pass done (main -> side)
    cudaEvent_t ev_xchg = nullptr;   // halos of the next pass received (side -> main)
};

namespace {

struct Nccl {
    bool ok = false;
    ncclResult_t (*GetUniqueId)(ncclUniqueId*) = nullptr;
    ncclResult_t (*CommInitRank)(ncclComm_t*, int, ncclUniqueId, int) = nullptr;
    ncclResult_t (*CommDestroy)(ncclComm_t) = nullptr;
    ncclResult_t (*Send)(const void*, size_t, ncclDataType_t, int, ncclComm_t, cudaStream_t) = nullptr;
    ncclResult_t (*Recv)(void*, size_t, ncclDataType_t, int, ncclComm_t, cudaStream_t) = nullptr;
    ncclResult_t (*GroupStart)() = nullptr;
    ncclResult_t (*GroupEnd)() = nullptr;
    ncclResult_t (*AllGather)(const void*, void*, size_t, ncclDataType_t, ncclComm_t, cudaStream_t) = nullptr;
    ncclResult_t (*CommGetAsyncError)(ncclComm_t, ncclResult_t*) = nullptr;
    ncclResult_t (*Broadcast)(const void*, void*, size_t, ncclDataType_t, int, ncclComm_t, cudaStream_t) = nullptr;
    ncclResult_t (*CommAbort)(ncclComm_t) = nullptr;
};

Nccl& nccl() {
    static Nccl n;
    static std::once_flag once;
    std::call_once(once, [] {
        void* h = nullptr;
        if (const char* p = std::getenv("SP_NCCL_LIB")) h = dlopen(p, RTLD_NOW | RTLD_GLOBAL);
        if (!h) h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_GLOBAL);
        if (!h) h = dlopen("libnccl.so", RTLD_NOW | RTLD_GLOBAL);
        if (!h) return;
#define SP_SYM(field, name) n.field = reinterpret_cast<decltype(n.field)>(dlsym(h, name))
        SP_SYM(GetUniqueId, "ncclGetUniqueId");
        SP_SYM(CommInitRank, "ncclCommInitRank");
        SP_SYM(CommDestroy, "ncclCommDestroy");
        SP_SYM(Send, "ncclSend");
        SP_SYM(Recv, "ncclRecv");
        SP_SYM(GroupStart, "ncclGroupStart");
        SP_SYM(GroupEnd, "ncclGroupEnd");
        SP_SYM(AllGather, "ncclAllGather");
        SP_SYM(CommGetAsyncError, "ncclCommGetAsyncError");
        SP_SYM(Broadcast, "ncclBroadcast");
        SP_SYM(CommAbort, "ncclCommAbort");
#undef SP_SYM
        n.ok = n.GetUniqueId && n.CommInitRank && n.CommDestroy && n.Send && n.Recv && n.GroupStart && n.GroupEnd &&
               n.AllGather;
    });
    return n;
}

#define SP_NCCL_TRY(expr)                      \
    do {                                       \
        ncclResult_t sp_r_ = (expr);           \
        if (sp_r_ != ncclSuccess) {            \
            sp::set_nccl_error((int)sp_r_);    \
            return SP_ERR_NCCL;                \
        }                                      \
    } while (0)

inline int32_t halo_of(int32_t tt) { return (tt + 3) & ~3; }

// One slab of the distributed domain.
struct Slab {
    float* a;  // holds global [x_begin - H, x_end + H)
    float* w;
    int64_t x_begin, n_local;
};

// Halo transport: exchange(cur_buffers) must fill, for every slab, the H cells on each side
// that belong to a neighbour's owned range.
template <class Exchange>
int pass_loop(std::vector<Slab>& slabs, int64_t n_global, int32_t steps, int32_t tt, int32_t space_tile,
              cudaStream_t stream, Exchange&& exchange) {
    const int32_t H = halo_of(tt);
    std::vector<float*> cur(slabs.size()), nxt(slabs.size());
    for (size_t r = 0; r < slabs.size(); ++r) {
        cur[r] = slabs[r].a;
        nxt[r] = slabs[r].w;
    }
    int st;
    for (int32_t done = 0; done < steps; done += tt) {
        const int32_t h = steps - done < tt ? steps - done : tt;
        {
            SP_NVTX("halo exchange");
            if ((st = exchange(cur))) return st;
        }
        for (size_t r = 0; r < slabs.size(); ++r) {
            const Slab& s = slabs[r];
            const int64_t g0 = s.x_begin - H;
            if ((st = sp_jacobi1d_pass_segment(cur[r], nxt[r], n_global, g0, s.n_local + 2 * H, s.x_begin,
                                               s.x_begin + s.n_local, h, tt, space_tile, stream)))
                return st;
        }
        std::swap(cur, nxt);
    }
    for (size_t r = 0; r < slabs.size(); ++r)
        if (cur[r] != slabs[r].a && slabs[r].n_local > 0)
            SP_CUDA_TRY(cudaMemcpyAsync(slabs[r].a + H, cur[r] + H, slabs[r].n_local * sizeof(float),
                                        cudaMemcpyDeviceToDevice, stream));
    return SP_OK;
}

int check_slab(int64_t n_global, int64_t x_begin, int64_t n_local, int32_t tt, const float* a, const float* w) {
    if (!a || !w || a == w || n_global < 3 || x_begin < 0 || n_local < 0 || x_begin + n_local > n_global)
        return SP_ERR_INVALID_ARG;
    if (tt < 1 || tt > 128) return SP_ERR_INVALID_ARG;
    if ((x_begin & 3) || (reinterpret_cast<uintptr_t>(a) & 15) || (reinterpret_cast<uintptr_t>(w) & 15))
        return SP_ERR_INVALID_ARG;
    return SP_OK;
}

}  // namespace

extern "C" int sp_get_unique_id(uint8_t out_id[128]) {
    if (!out_id) return SP_ERR_INVALID_ARG;
    Nccl& n = nccl();
    if (!n.ok) {
        sp::set_nccl_error((int)ncclSystemError);
        return SP_ERR_NCCL;
    }
    ncclUniqueId id;
    SP_NCCL_TRY(n.GetUniqueId(&id));
    std::memcpy(out_id, id.internal, 128);
    return SP_OK;
}

extern "C" int sp_comm_init(sp_comm** out, const uint8_t id[128], int32_t nranks, int32_t rank, int32_t device) {
    if (!out || !id || nranks < 1 || rank < 0 || rank >= nranks || device < 0) return SP_ERR_INVALID_ARG;
    Nccl& n = nccl();
    if (!n.ok) {
        sp::set_nccl_error((int)ncclSystemError);
        return SP_ERR_NCCL;
    }
    SP_CUDA_TRY(cudaSetDevice(device));
    ncclUniqueId uid;
    std::memcpy(uid.internal, id, 128);
    sp_comm* c = new sp_comm;
    c->rank = rank;
    c->nranks = nranks;
    c->device = device;
    ncclResult_t r = n.CommInitRank(&c->comm, nranks, uid, rank);
    if (r != ncclSuccess) {
        delete c;
        sp::set_nccl_error((int)r);
        return SP_ERR_NCCL;
    }
    if (cudaStreamCreateWithFlags(&c->side, cudaStreamNonBlocking) != cudaSuccess ||
        cudaEventCreateWithFlags(&c->ev_edge, cudaEventDisableTiming) != cudaSuccess ||
        cudaEventCreateWithFlags(&c->ev_xchg, cudaEventDisableTiming) != cudaSuccess) {
        sp::set_cuda_error((int)cudaGetLastError());
        n.CommDestroy(c->comm);
        delete c;
        return SP_ERR_CUDA;
    }
    *out = c;
    return SP_OK;
}

extern "C" int sp_comm_destroy(sp_comm* c) {
    if (!c) return SP_ERR_INVALID_ARG;
    if (c->side) cudaStreamDestroy(c->side);
    if (c->ev_edge) cudaEventDestroy(c->ev_edge);
    if (c->ev_xchg) cudaEventDestroy(c->ev_xchg);
    Nccl& n = nccl();
    if (c->comm && n.ok) {
        ncclResult_t r = n.CommDestroy(c->comm);
        delete c;
        if (r != ncclSuccess) {
            sp::set_nccl_error((int)r);
            return SP_ERR_NCCL;
        }
        return SP_OK;
    }
    delete c;
    return SP_OK;
}

namespace {
// asynchronous NCCL failure of the communicator (anything but success / in progress)
int check_async(sp_comm* c) {
    Nccl& n = nccl();
    if (!n.CommGetAsyncError) return SP_OK;
    ncclResult_t r = ncclSuccess;
    SP_NCCL_TRY(n.CommGetAsyncError(c->comm, &r));
    if (r != ncclSuccess && r != ncclInProgress) {
        sp::set_nccl_error((int)r);
        return SP_ERR_NCCL;
    }
    return SP_OK;
}
}  // namespace

// NCCL baseline of the multi-GPU Jacobi (the fused peer-memory kernel is the product path):
// per pass the slab's two EDGE segments (the first / last H owned cells — the only cells a
// neighbour reads) run first, the halo exchange of the next pass (grouped ncclSend/ncclRecv)
// then runs on a side stream while the INTERIOR segment computes on `stream`, and the next
// pass waits for the exchange (the per-time-tile synchronisation, here
// overlapped with the interior work).  Buffer positions: b[j] <-> global x_begin - H + j; the
// edge / interior kernels write disjoint owned cells, the exchange reads the new edge cells and
// writes only halo cells, so nothing races.
extern "C" int sp_jacobi1d_timetiled_dist(sp_comm* c, float* a_local, float* work_local, int64_t n_global,
                                          int64_t x_begin, int64_t n_local, int32_t steps, int32_t time_tile,
                                          int32_t space_tile, void* stream) {
    SP_NVTX("sp_jacobi1d_timetiled_dist");
    if (!c) return SP_ERR_INVALID_ARG;
    int st = check_slab(n_global, x_begin, n_local, time_tile, a_local, work_local);
    if (st) return st;
    const int32_t H = halo_of(time_tile);
    if (steps < 0 || (c->nranks > 1 && n_local < H)) return SP_ERR_INVALID_ARG;
    if (steps == 0) return SP_OK;
    Nccl& n = nccl();
    const cudaStream_t s = (cudaStream_t)stream;
    const int64_t x_end = x_begin + n_local;
    const int left = (x_begin > 0) ? c->rank - 1 : -1;
    const int right = (x_end < n_global) ? c->rank + 1 : -1;
    const int64_t g0 = x_begin - H, len = n_local + 2 * H;
    auto exchange = [&](float* b, cudaStream_t q) -> int {  // b's halos <- the neighbours' edge cells
        if (left < 0 && right < 0) return SP_OK;
        SP_NCCL_TRY(n.GroupStart());
        if (left >= 0) {
            SP_NCCL_TRY(n.Send(b + H, H, ncclFloat32, left, c->comm, q));  // my first H owned cells
            SP_NCCL_TRY(n.Recv(b, H, ncclFloat32, left, c->comm, q));      // left halo
        }
        if (right >= 0) {
            SP_NCCL_TRY(n.Send(b + n_local, H, ncclFloat32, right, c->comm, q));  // my last H owned
            SP_NCCL_TRY(n.Recv(b + H + n_local, H, ncclFloat32, right, c->comm, q));
        }
        SP_NCCL_TRY(n.GroupEnd());
        return check_async(c);
    };
    auto segment = [&](float* src, float* dst, int64_t ob, int64_t oe, int32_t h) -> int {
        if (oe <= ob) return SP_OK;
        return sp_jacobi1d_pass_segment(src, dst, n_global, g0, len, ob, oe, h, time_tile, space_tile, stream);
    };
    // edges split off only when an interior remains (and a neighbour exists)
    const bool split = (left >= 0 || right >= 0) && n_local >= 3 * (int64_t)H;
    const int64_t ib = left >= 0 ? x_begin + H : x_begin, ie = right >= 0 ? x_end - H : x_end;
    float* cur = a_local;
    float* nxt = work_local;
    {
        SP_NVTX("halo exchange");
        if ((st = exchange(cur, s))) return st;
    }
    for (int32_t done = 0; done < steps; done += time_tile) {
        const int32_t h = steps - done < time_tile ? steps - done : time_tile;
        const bool more = done + time_tile < steps;
        if (!split) {
            if ((st = segment(cur, nxt, x_begin, x_end, h))) return st;
            if (more && (st = exchange(nxt, s))) return st;
        } else {
            if (left >= 0 && (st = segment(cur, nxt, x_begin, x_begin + H, h))) return st;
            if (right >= 0 && (st = segment(cur, nxt, x_end - H, x_end, h))) return st;
            if (more) {
                SP_CUDA_TRY(cudaEventRecord(c->ev_edge, s));
                SP_CUDA_TRY(cudaStreamWaitEvent(c->side, c->ev_edge, 0));
                {
                    SP_NVTX("halo exchange (overlapped)");
                    if ((st = exchange(nxt, c->side))) return st;
                }
                SP_CUDA_TRY(cudaEventRecord(c->ev_xchg, c->side));
            }
            if ((st = segment(cur, nxt, ib, ie, h))) return st;
            if (more) SP_CUDA_TRY(cudaStreamWaitEvent(s, c->ev_xchg, 0));
        }
        std::swap(cur, nxt);
    }
    if (cur != a_local && n_local > 0)
        SP_CUDA_TRY(cudaMemcpyAsync(a_local + H, cur + H, n_local * sizeof(float), cudaMemcpyDeviceToDevice, s));
    return SP_OK;
}

// Failure detection with a deadline: wait for `stream` while polling the communicator's
// asynchronous error; on an NCCL error or when timeout_ms passes first (a peer died or hangs),
// the communicator is aborted (ncclCommAbort: its kernels return) and SP_ERR_NCCL is returned
// (sp_last_nccl_error: the NCCL error, or ncclInProgress = 7 for a timeout).
extern "C" int sp_comm_sync(sp_comm* c, void* stream, int64_t timeout_ms) {
    if (!c || timeout_ms < 0) return SP_ERR_INVALID_ARG;
    Nccl& n = nccl();
    const auto t0 = std::chrono::steady_clock::now();
    for (;;) {
        const cudaError_t q = cudaStreamQuery((cudaStream_t)stream);
        if (q == cudaSuccess) return SP_OK;
        if (q != cudaErrorNotReady) {
            sp::set_cuda_error((int)q);
            return SP_ERR_CUDA;
        }
        ncclResult_t r = ncclSuccess;
        if (n.CommGetAsyncError && n.CommGetAsyncError(c->comm, &r) == ncclSuccess && r != ncclSuccess &&
            r != ncclInProgress) {
            if (n.CommAbort) n.CommAbort(c->comm);
            c->comm = nullptr;
            sp::set_nccl_error((int)r);
            return SP_ERR_NCCL;
        }
        if (std::chrono::steady_clock::now() - t0 > std::chrono::milliseconds(timeout_ms)) {
            if (n.CommAbort) n.CommAbort(c->comm);
            c->comm = nullptr;
            sp::set_nccl_error((int)ncclInProgress);
            return SP_ERR_NCCL;
        }
        std::this_thread::sleep_for(std::chrono::microseconds(100));
    }
}

extern "C" int sp_comm_async_error(sp_comm* c, int32_t* nccl_result) {
    if (!c || !nccl_result) return SP_ERR_INVALID_ARG;
    Nccl& n = nccl();
    if (!n.ok || !n.CommGetAsyncError) {
        sp::set_nccl_error((int)ncclSystemError);
        return SP_ERR_NCCL;
    }
    ncclResult_t r = ncclSuccess;
    SP_NCCL_TRY(n.CommGetAsyncError(c->comm, &r));
    *nccl_result = (int32_t)r;
    return SP_OK;
}

extern "C" int sp_allgather(sp_comm* c, const void* send, void* recv, int64_t bytes, void* stream) {
    SP_NVTX("sp_allgather");
    if (!c || !send || !recv || bytes < 0) return SP_ERR_INVALID_ARG;
    Nccl& n = nccl();
    SP_NCCL_TRY(n.AllGather(send, recv, (size_t)bytes, ncclUint8, c->comm, (cudaStream_t)stream));
    return SP_OK;
}

// Single-GPU loopback transport of the same partitioned pass loop (test vehicle for the
// decomposition and for the overlapped schedule of sp_jacobi1d_timetiled_dist; not a performance
// path).  Slab r owns [x_begins[r], x_begins[r] + n_locals[r]); slabs must tile [0, n_global) in
// order.  Per pass: every slab's edge segments, then the halo copies on a side stream while the
// interior segments run on `stream` (the exchange of the dist path, with cudaMemcpyAsync in
// place of ncclSend/ncclRecv).
extern "C" int sp_jacobi1d_timetiled_loopback(float** a_locals, float** work_locals, int32_t nranks, int64_t n_global,
                                              const int64_t* x_begins, const int64_t* n_locals, int32_t steps,
                                              int32_t time_tile, int32_t space_tile, void* stream) {
    SP_NVTX("sp_jacobi1d_timetiled_loopback");
    if (!a_locals || !work_locals || !x_begins || !n_locals || nranks < 1) return SP_ERR_INVALID_ARG;
    const int32_t H = halo_of(time_tile);
    std::vector<Slab> slabs;
    int64_t expect = 0;
    for (int r = 0; r < nranks; ++r) {
        int st = check_slab(n_global, x_begins[r], n_locals[r], time_tile, a_locals[r], work_locals[r]);
        if (st) return st;
        if (x_begins[r] != expect || (nranks > 1 && n_locals[r] < H)) return SP_ERR_INVALID_ARG;
        expect += n_locals[r];
        slabs.push_back({a_locals[r], work_locals[r], x_begins[r], n_locals[r]});
    }
    if (expect != n_global || steps < 0) return SP_ERR_INVALID_ARG;
    if (steps == 0) return SP_OK;
    const cudaStream_t s = (cudaStream_t)stream;
    cudaStream_t side = nullptr;
    cudaEvent_t ev_edge = nullptr, ev_xchg = nullptr;
    SP_CUDA_TRY(cudaStreamCreateWithFlags(&side, cudaStreamNonBlocking));
    SP_CUDA_TRY(cudaEventCreateWithFlags(&ev_edge, cudaEventDisableTiming));
    SP_CUDA_TRY(cudaEventCreateWithFlags(&ev_xchg, cudaEventDisableTiming));
    std::vector<float*> cur(nranks), nxt(nranks);
    for (int r = 0; r < nranks; ++r) {
        cur[r] = slabs[r].a;
        nxt[r] = slabs[r].w;
    }
    auto exchange = [&](std::vector<float*>& b, cudaStream_t q) -> int {
        for (int r = 0; r < nranks; ++r) {
            const int64_t nl = slabs[r].n_local;
            if (r > 0)  // left halo <- left neighbour's last H owned cells
                SP_CUDA_TRY(cudaMemcpyAsync(b[r], b[r - 1] + slabs[r - 1].n_local, H * sizeof(float),
                                            cudaMemcpyDeviceToDevice, q));
            if (r + 1 < nranks)  // right halo <- right neighbour's first H owned cells
                SP_CUDA_TRY(cudaMemcpyAsync(b[r] + H + nl, b[r + 1] + H, H * sizeof(float), cudaMemcpyDeviceToDevice,
                                            q));
        }
        return SP_OK;
    };
    auto segment = [&](int r, int64_t ob, int64_t oe, int32_t h) -> int {
        if (oe <= ob) return SP_OK;
        const Slab& sl = slabs[r];
        return sp_jacobi1d_pass_segment(cur[r], nxt[r], n_global, sl.x_begin - H, sl.n_local + 2 * H, ob, oe, h,
                                        time_tile, space_tile, s);
    };
    int st = exchange(cur, s);
    for (int32_t done = 0; st == SP_OK && done < steps; done += time_tile) {
        const int32_t h = steps - done < time_tile ? steps - done : time_tile;
        const bool more = done + time_tile < steps;
        std::vector<char> split(nranks);
        // 1. edge segments of split slabs, whole unsplit slabs
        for (int r = 0; r < nranks && st == SP_OK; ++r) {
            const Slab& sl = slabs[r];
            const int64_t xe = sl.x_begin + sl.n_local;
            split[r] = nranks > 1 && sl.n_local >= 3 * (int64_t)H;
            if (!split[r]) {
                st = segment(r, sl.x_begin, xe, h);
                continue;
            }
            if (r > 0) st = segment(r, sl.x_begin, sl.x_begin + H, h);
            if (st == SP_OK && r + 1 < nranks) st = segment(r, xe - H, xe, h);
        }
        if (st) break;
        // 2. the next pass's halos on the side stream, after every edge cell exists
        if (more) {
            if (cudaEventRecord(ev_edge, s) != cudaSuccess || cudaStreamWaitEvent(side, ev_edge, 0) != cudaSuccess) {
                st = SP_ERR_CUDA;
                break;
            }
            if ((st = exchange(nxt, side))) break;
            if (cudaEventRecord(ev_xchg, side) != cudaSuccess) {
                st = SP_ERR_CUDA;
                break;
            }
        }
        // 3. interiors of split slabs, concurrently with the exchange
        for (int r = 0; r < nranks && st == SP_OK; ++r) {
            if (!split[r]) continue;
            const Slab& sl = slabs[r];
            const int64_t xe = sl.x_begin + sl.n_local;
            st = segment(r, r > 0 ? sl.x_begin + H : sl.x_begin, r + 1 < nranks ? xe - H : xe, h);
        }
        if (st) break;
        if (more && cudaStreamWaitEvent(s, ev_xchg, 0) != cudaSuccess) st = SP_ERR_CUDA;
        std::swap(cur, nxt);
    }
    for (int r = 0; st == SP_OK && r < nranks; ++r)
        if (cur[r] != slabs[r].a && slabs[r].n_local > 0 &&
            cudaMemcpyAsync(slabs[r].a + H, cur[r] + H, slabs[r].n_local * sizeof(float), cudaMemcpyDeviceToDevice,
                            s) != cudaSuccess)
            st = SP_ERR_CUDA;
    if (st == SP_ERR_CUDA) sp::set_cuda_error((int)cudaGetLastError());
    cudaEventDestroy(ev_edge);
    cudaEventDestroy(ev_xchg);
    cudaStreamDestroy(side);  // (destroy after pending work: resources are released on completion)
    return st;
}

// NCCL baseline of the ME all-gather (the fused peer-store gather of sp_me_sad_search_gather is
// the product path): this rank's range, then one ncclBroadcast per rank and output array, each
// rank the root of its own range, in place in the global arrays (an all-gather-v).
extern "C" int sp_me_sad_search_dist(sp_comm* c, const uint8_t* ref, const uint8_t* cur, int64_t pitch, int32_t width,
                                     int32_t frame_height, int32_t n_pairs_buffer, int64_t pair_stride,
                                     int32_t pair_base, int32_t range, const int64_t* flat_ranges, int16_t* mv,
                                     uint32_t* best_sad, void* stream) {
    SP_NVTX("sp_me_sad_search_dist");
    if (!c || !flat_ranges || !mv || !best_sad) return SP_ERR_INVALID_ARG;
    for (int q = 0; q < c->nranks; ++q)
        if (flat_ranges[2 * q] > flat_ranges[2 * q + 1] || (q > 0 && flat_ranges[2 * q] != flat_ranges[2 * q - 1]))
            return SP_ERR_INVALID_ARG;
    int st = sp_me_sad_search_range(ref, cur, pitch, width, frame_height, n_pairs_buffer, pair_stride, pair_base, range,
                                    flat_ranges[2 * c->rank], flat_ranges[2 * c->rank + 1], mv, best_sad, stream);
    if (st) return st;
    if (c->nranks == 1) return SP_OK;
    Nccl& n = nccl();
    if (!n.Broadcast) {
        sp::set_nccl_error((int)ncclSystemError);
        return SP_ERR_NCCL;
    }
    const int64_t mbx = width / 16;
    const cudaStream_t s = (cudaStream_t)stream;
    SP_NCCL_TRY(n.GroupStart());
    for (int q = 0; q < c->nranks; ++q) {
        const int64_t off = flat_ranges[2 * q] * mbx, cnt = (flat_ranges[2 * q + 1] - flat_ranges[2 * q]) * mbx;
        if (cnt == 0) continue;
        SP_NCCL_TRY(n.Broadcast(mv + 2 * off, mv + 2 * off, (size_t)(4 * cnt), ncclUint8, q, c->comm, s));
        SP_NCCL_TRY(n.Broadcast(best_sad + off, best_sad + off, (size_t)(4 * cnt), ncclUint8, q, c->comm, s));
    }
    SP_NCCL_TRY(n.GroupEnd());
    return check_async(c);
}

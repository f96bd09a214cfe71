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

#include <cstdlib>
#include <cstring>
#include <mutex>
#include <vector>

#include "../../include/sp.h"
#include "sp_internal.h"
#include "sp_nccl_min.h"

struct sp_comm {
    ncclComm_t comm = nullptr;
    int32_t rank = 0, nranks = 1, device = 0;
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
    *out = c;
    return SP_OK;
}

extern "C" int sp_comm_destroy(sp_comm* c) {
    if (!c) return SP_ERR_INVALID_ARG;
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
    std::vector<Slab> slabs{{a_local, work_local, x_begin, n_local}};
    const int64_t x_end = x_begin + n_local;
    const int left = (x_begin > 0) ? c->rank - 1 : -1;
    const int right = (x_end < n_global) ? c->rank + 1 : -1;
    return pass_loop(slabs, n_global, steps, time_tile, space_tile, s, [&](std::vector<float*>& cur) -> int {
        if (left < 0 && right < 0) return SP_OK;
        float* b = cur[0];  // b[j] <-> global x_begin - H + j
        SP_NCCL_TRY(n.GroupStart());
        if (left >= 0) {
            SP_NCCL_TRY(n.Send(b + H, H, ncclFloat32, left, c->comm, s));  // my first H owned cells
            SP_NCCL_TRY(n.Recv(b, H, ncclFloat32, left, c->comm, s));      // left halo
        }
        if (right >= 0) {
            SP_NCCL_TRY(n.Send(b + n_local, H, ncclFloat32, right, c->comm, s));  // my last H owned
            SP_NCCL_TRY(n.Recv(b + H + n_local, H, ncclFloat32, right, c->comm, s));
        }
        SP_NCCL_TRY(n.GroupEnd());
        return SP_OK;
    });
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
// decomposition; not a performance path).  Slab r owns [x_begins[r], x_begins[r] +
// n_locals[r]); slabs must tile [0, n_global) in order.
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
    return pass_loop(slabs, n_global, steps, time_tile, space_tile, s, [&](std::vector<float*>& cur) -> int {
        for (int r = 0; r < nranks; ++r) {
            const int64_t nl = slabs[r].n_local;
            if (r > 0)  // left halo <- left neighbour's last H owned cells
                SP_CUDA_TRY(cudaMemcpyAsync(cur[r], cur[r - 1] + slabs[r - 1].n_local, H * sizeof(float),
                                            cudaMemcpyDeviceToDevice, s));
            if (r + 1 < nranks)  // right halo <- right neighbour's first H owned cells
                SP_CUDA_TRY(cudaMemcpyAsync(cur[r] + H + nl, cur[r + 1] + H, H * sizeof(float),
                                            cudaMemcpyDeviceToDevice, s));
        }
        return SP_OK;
    });
}

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
    return SP_OK;
}

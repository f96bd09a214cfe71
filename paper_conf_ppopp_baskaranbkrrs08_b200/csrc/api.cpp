// api.cpp — status strings, version, thread-local error slots of the libsp C ABI.
#include "../../include/sp.h"
#include "sp_internal.h"

namespace sp {
static thread_local int g_cuda_error = 0;
static thread_local int g_nccl_error = 0;
void set_cuda_error(int e) { g_cuda_error = e; }
void set_nccl_error(int e) { g_nccl_error = e; }
}  // namespace sp

extern "C" const char* sp_status_string(int status) {
    switch (status) {
        case SP_OK: return "SP_OK";
        case SP_ERR_INVALID_ARG: return "SP_ERR_INVALID_ARG";
        case SP_ERR_UNBOUNDED: return "SP_ERR_UNBOUNDED";
        case SP_ERR_CAPACITY: return "SP_ERR_CAPACITY";
        case SP_ERR_OVERFLOW: return "SP_ERR_OVERFLOW";
        case SP_ERR_UNSUPPORTED: return "SP_ERR_UNSUPPORTED";
        case SP_ERR_SMEM_LIMIT: return "SP_ERR_SMEM_LIMIT";
        case SP_ERR_CUDA: return "SP_ERR_CUDA";
        case SP_ERR_NCCL: return "SP_ERR_NCCL";
        default: return "SP_ERR_UNKNOWN";
    }
}
extern "C" int sp_last_cuda_error(void) { return sp::g_cuda_error; }
extern "C" int sp_last_nccl_error(void) { return sp::g_nccl_error; }
extern "C" int sp_version(void) { return 100; }
extern "C" int sp_abi_struct_sizes(int64_t* out, int32_t n) {
    const int64_t sz[] = {sizeof(sp_domain),      sizeof(sp_ref),         sizeof(sp_block),      sizeof(sp_plan_opts),
                          sizeof(sp_buffer),      sizeof(sp_jacobi_plan), sizeof(sp_peer_links), sizeof(sp_tile_problem),
                          sizeof(sp_tile_result), sizeof(sp_op),          sizeof(sp_stmt_body),  sizeof(sp_array_desc),
                          sizeof(sp_exec_opts),   sizeof(sp_exec_stats), sizeof(sp_me_gather_links)};
    const int32_t k = (int32_t)(sizeof(sz) / sizeof(sz[0]));
    for (int32_t i = 0; out && i < n && i < k; ++i) out[i] = sz[i];
    return k;
}

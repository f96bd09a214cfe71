// sp_internal.h — private helpers shared by the libsp translation units.
#pragma once
#include <cstdint>
#include <vector>

#include <nvtx3/nvToolsExt.h>

#include "../../include/sp.h"

namespace sp {
// integer points of a statement domain with concrete parameters, lexicographic loop order,
// appended to `out` as depth-long vectors, their number in *count (planner.cpp; used by
// the executor, exec.cu)
int enumerate_domain(const sp_domain& D, int n_params, const int64_t* params, int64_t max_points,
                     std::vector<int64_t>& out, int64_t* count);
// thread-local last CUDA / NCCL error (see sp_last_cuda_error / sp_last_nccl_error)
void set_cuda_error(int e);
void set_nccl_error(int e);
}  // namespace sp

#define SP_CUDA_TRY(expr)                                 \
    do {                                                  \
        cudaError_t sp_e_ = (expr);                       \
        if (sp_e_ != cudaSuccess) {                       \
            sp::set_cuda_error((int)sp_e_);               \
            return SP_ERR_CUDA;                           \
        }                                                 \
    } while (0)

// NVTX range over an entry point (SURVEY §5 tracing): visible to ncu (--nvtx) and nsys;
// header-only NVTX v3, a no-op unless a tool is attached.
namespace sp {
struct NvtxRange {
    explicit NvtxRange(const char* name) { nvtxRangePushA(name); }
    ~NvtxRange() { nvtxRangePop(); }
    NvtxRange(const NvtxRange&) = delete;
    NvtxRange& operator=(const NvtxRange&) = delete;
};
}  // namespace sp
#define SP_NVTX(name) const sp::NvtxRange sp_nvtx_range_(name)

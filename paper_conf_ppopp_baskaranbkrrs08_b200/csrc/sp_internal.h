// sp_internal.h — private helpers shared by the libsp translation units.
#pragma once
#include <cstdint>

namespace sp {
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

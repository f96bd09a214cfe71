// Probe: 1-D bulk TMA (cp.async.bulk) straight from / to pinned host memory (zero copy over
// PCIe), against cudaMemcpyAsync.  Decides whether the host-buffer Jacobi/ME entry points can
// stream their inputs and outputs through the kernels' own move-in / move-out.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o sysmem_tma_probe sysmem_tma_probe.cu
#include <cuda_runtime.h>
#include <cstdint>
#include <cstdio>
#include <cstring>

__device__ __forceinline__ uint32_t sa(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }

// each warp copies chunks of `chunk` bytes src -> smem -> dst with bulk TMA (load + store)
__global__ void __launch_bounds__(256) copy_kernel(const uint8_t* src, uint8_t* dst, size_t bytes, int chunk) {
    extern __shared__ __align__(128) uint8_t sm[];
    __shared__ __align__(8) uint64_t bar[8];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    uint8_t* buf = sm + warp * chunk;
    if (lane == 0) {
        asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(sa(&bar[warp])));
        asm volatile("fence.mbarrier_init.release.cluster;");
    }
    __syncwarp();
    const size_t nchunks = bytes / chunk;
    uint32_t ph = 0;
    for (size_t c = (size_t)blockIdx.x * 8 + warp; c < nchunks; c += (size_t)gridDim.x * 8) {
        if (lane == 0) {
            asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");
            asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(sa(&bar[warp])), "r"(chunk));
            asm volatile(
                "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(sa(buf)),
                "l"(src + c * chunk), "r"(chunk), "r"(sa(&bar[warp]))
                : "memory");
            asm volatile(
                "{\n\t.reg .pred p;\n\tW: mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t@!p bra W;\n\t}" ::"r"(
                    sa(&bar[warp])),
                "r"(ph)
                : "memory");
            asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(dst + c * chunk),
                         "r"(sa(buf)), "r"(chunk)
                         : "memory");
            asm volatile("cp.async.bulk.commit_group;" ::: "memory");
        }
        ph ^= 1;
        __syncwarp();
    }
    if (lane == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
}

#define CK(x)                                                                              \
    do {                                                                                   \
        cudaError_t e_ = (x);                                                              \
        if (e_ != cudaSuccess) {                                                           \
            printf("FAIL %s: %s (line %d)\n", #x, cudaGetErrorString(e_), __LINE__);       \
            return 1;                                                                      \
        }                                                                                  \
    } while (0)

int main() {
    const size_t bytes = (size_t)256 << 20;
    const int chunk = 7168;
    uint8_t *h_in, *h_out, *d_a, *d_b;
    CK(cudaHostAlloc(&h_in, bytes, cudaHostAllocMapped | cudaHostAllocPortable));
    CK(cudaHostAlloc(&h_out, bytes, cudaHostAllocMapped | cudaHostAllocPortable));
    CK(cudaMalloc(&d_a, bytes));
    CK(cudaMalloc(&d_b, bytes));
    for (size_t i = 0; i < bytes; ++i) h_in[i] = (uint8_t)(i * 2654435761u >> 13);
    memset(h_out, 0, bytes);
    CK(cudaFuncSetAttribute(copy_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 8 * chunk));
    cudaEvent_t e0, e1;
    CK(cudaEventCreate(&e0));
    CK(cudaEventCreate(&e1));
    float ms;
    const size_t nb = bytes / chunk * chunk;
    for (int grid : {148, 296}) {
        for (int rep = 0; rep < 3; ++rep) {
            CK(cudaEventRecord(e0));
            copy_kernel<<<grid, 256, 8 * chunk>>>(h_in, d_a, bytes, chunk);  // host -> device by TMA
            CK(cudaEventRecord(e1));
            CK(cudaEventSynchronize(e1));
            CK(cudaGetLastError());
            CK(cudaEventElapsedTime(&ms, e0, e1));
            printf("TMA host->dev grid %d: %.3f ms  %.1f GB/s\n", grid, ms, nb / ms / 1e6);
        }
        for (int rep = 0; rep < 3; ++rep) {
            CK(cudaEventRecord(e0));
            copy_kernel<<<grid, 256, 8 * chunk>>>(d_a, h_out, bytes, chunk);  // device -> host by TMA
            CK(cudaEventRecord(e1));
            CK(cudaEventSynchronize(e1));
            CK(cudaGetLastError());
            CK(cudaEventElapsedTime(&ms, e0, e1));
            printf("TMA dev->host grid %d: %.3f ms  %.1f GB/s\n", grid, ms, nb / ms / 1e6);
        }
    }
    size_t bad = 0;
    for (size_t i = 0; i < nb; ++i) bad += h_out[i] != h_in[i];
    printf("round trip mismatches: %zu\n", bad);
    cudaStream_t s1, s2;
    CK(cudaStreamCreateWithFlags(&s1, cudaStreamNonBlocking));
    CK(cudaStreamCreateWithFlags(&s2, cudaStreamNonBlocking));
    for (int rep = 0; rep < 3; ++rep) {
        CK(cudaEventRecord(e0));
        CK(cudaMemcpyAsync(d_b, h_in, bytes, cudaMemcpyHostToDevice, 0));
        CK(cudaEventRecord(e1));
        CK(cudaEventSynchronize(e1));
        CK(cudaEventElapsedTime(&ms, e0, e1));
        printf("memcpy H2D: %.3f ms  %.1f GB/s\n", ms, bytes / ms / 1e6);
        CK(cudaEventRecord(e0));
        CK(cudaMemcpyAsync(h_out, d_b, bytes, cudaMemcpyDeviceToHost, 0));
        CK(cudaEventRecord(e1));
        CK(cudaEventSynchronize(e1));
        CK(cudaEventElapsedTime(&ms, e0, e1));
        printf("memcpy D2H: %.3f ms  %.1f GB/s\n", ms, bytes / ms / 1e6);
    }
    // both directions at once: TMA kernels on two streams
    for (int rep = 0; rep < 3; ++rep) {
        CK(cudaDeviceSynchronize());
        CK(cudaEventRecord(e0, s1));
        CK(cudaStreamWaitEvent(s2, e0));
        copy_kernel<<<74, 256, 8 * chunk, s1>>>(h_in, d_a, bytes, chunk);
        copy_kernel<<<74, 256, 8 * chunk, s2>>>(d_b, h_out, bytes, chunk);
        cudaEvent_t e2;
        CK(cudaEventCreate(&e2));
        CK(cudaEventRecord(e2, s2));
        CK(cudaStreamWaitEvent(s1, e2));
        CK(cudaEventRecord(e1, s1));
        CK(cudaEventSynchronize(e1));
        CK(cudaGetLastError());
        CK(cudaEventElapsedTime(&ms, e0, e1));
        printf("TMA both directions (74+74 CTAs): %.3f ms  %.1f GB/s each way\n", ms, nb / ms / 1e6);
    }
    printf("probe done\n");
    return 0;
}

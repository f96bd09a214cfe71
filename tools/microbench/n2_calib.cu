// N2 calibration: the two constants of the paper's movement
// cost model C = N (P S + V L / P), measured on this GPU for the mechanisms the kernels use.
//
//  S — synchronisation cost per process per movement:
//      (a) CTA barrier (bar.sync) with P = 32..1024 threads: cycles per barrier / P;
//      (b) the persistent Jacobi's per-tile synchronisation: publish a finished tile
//          (fence.proxy.async + st.release.gpu of a flag) and a dependent warp on another SM
//          observing it (ld.relaxed poll + fence.acq_rel): one-way latency from a two-CTA
//          ping-pong; plus the unit-counter atomicAdd round trip;
//      (c) mbarrier wait of an already-complete TMA transaction.
//  L — cost of moving one element: 1-D bulk TMA (cp.async.bulk global -> shared, mbarrier
//      completion) of strips of the kernels' sizes from a 2 GiB HBM buffer (never L2-resident),
//      one CTA per SM (all SMs, HBM-bound) and one CTA alone (per-SM engine limit):
//      bytes per clock per SM.
// Output: one JSON object on stdout.  Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3
//   -o n2_calib n2_calib.cu -I ../../paper_conf_ppopp_baskaranbkrrs08_b200/csrc
#include <cuda_runtime.h>

#include <cstdint>
#include <cstdio>
#include <vector>

#include "sm100_ptx.cuh"

using namespace sp::ptx;

#define CK(x)                                                                            \
    do {                                                                                 \
        cudaError_t e_ = (x);                                                            \
        if (e_ != cudaSuccess) {                                                         \
            fprintf(stderr, "CUDA %s @%d\n", cudaGetErrorString(e_), __LINE__);          \
            return 1;                                                                    \
        }                                                                                \
    } while (0)

__device__ long long g_out[4096];

// (a) barrier latency: ITER bar.sync per CTA, cycles per barrier (thread 0's clock)
__global__ void bar_kernel(int iters) {
    __syncthreads();
    const long long t0 = clock64();
    for (int i = 0; i < iters; ++i) __syncthreads();
    const long long t1 = clock64();
    if (threadIdx.x == 0) g_out[blockIdx.x] = t1 - t0;
}

// (b) flag ping-pong between CTA 0 and CTA 1 (different SMs): CTA 0 publishes k, CTA 1 waits
// for k and publishes k back on a second flag.  Round trip / 2 = one-way publish -> observe.
__global__ void pingpong_kernel(int* flags, int iters) {
    if (threadIdx.x != 0) return;
    int* mine = flags + (blockIdx.x ? 32 : 0);
    int* theirs = flags + (blockIdx.x ? 0 : 32);
    const long long t0 = clock64();
    for (int k = 1; k <= iters; ++k) {
        if (blockIdx.x == 0) {
            fence_proxy_async_global();
            st_release_gpu(mine, k);
            while (ld_relaxed_gpu(theirs) < k) {
            }
            fence_acq_rel_gpu();
        } else {
            while (ld_relaxed_gpu(theirs) < k) {
            }
            fence_acq_rel_gpu();
            fence_proxy_async_global();
            st_release_gpu(mine, k);
        }
    }
    const long long t1 = clock64();
    if (blockIdx.x == 0) g_out[0] = t1 - t0;
}

// unit-counter atomic round trip (one thread, each atomic's address depends on the previous
// result, so the round trips cannot overlap)
__global__ void atomic_kernel(int* ctr, int iters) {
    if (threadIdx.x != 0) return;
    int v = 0;
    const long long t0 = clock64();
    for (int i = 0; i < iters; ++i) v = atomicAdd(ctr + ((unsigned)v >> 30), 1);
    const long long t1 = clock64();
    g_out[blockIdx.x] = t1 - t0 + (v == -1);
}

// (c) + L: per CTA, `chunks` consecutive bulk copies of `bytes` each from src (CTA-strided
// over a large buffer), double-buffered in shared memory, each waited on an mbarrier.
__global__ void tma_kernel(const uint8_t* src, size_t span, uint32_t bytes, int chunks) {
    extern __shared__ __align__(128) uint8_t smem[];
    __shared__ __align__(8) uint64_t bar[2];
    if (threadIdx.x != 0) return;
    mbar_init(&bar[0], 1);
    mbar_init(&bar[1], 1);
    fence_mbar_init();
    size_t off = ((size_t)blockIdx.x * chunks * bytes) % span;
    const long long t0 = clock64();
    mbar_arrive_expect_tx(&bar[0], bytes);
    tma_load_1d(smem, src + off, bytes, &bar[0]);
    long long wait_done = 0;
    for (int c = 0; c < chunks; ++c) {
        const int s = c & 1;
        if (c + 1 < chunks) {
            size_t o2 = off + (size_t)(c + 1) * bytes;
            if (o2 + bytes > span) o2 %= (span - bytes);
            o2 &= ~(size_t)15;
            mbar_arrive_expect_tx(&bar[s ^ 1], bytes);
            tma_load_1d(smem + (s ^ 1) * bytes, src + o2, bytes, &bar[s ^ 1]);
        }
        mbar_wait(&bar[s], (c >> 1) & 1);
        if (c == chunks - 1) {  // (c): a wait on an already-complete phase
            const long long w0 = clock64();
            for (int r = 0; r < 64; ++r) mbar_wait(&bar[s], (c >> 1) & 1);
            wait_done = (clock64() - w0) / 64;
        }
    }
    const long long t1 = clock64();
    g_out[blockIdx.x] = t1 - t0;
    if (blockIdx.x == 0) g_out[4095] = wait_done;
}

int main() {
    int sms = 0, clk_khz = 0;
    CK(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0));
    CK(cudaDeviceGetAttribute(&clk_khz, cudaDevAttrClockRate, 0));
    std::vector<long long> h(4096);
    printf("{\"sms\": %d, \"clock_khz_attr\": %d", sms, clk_khz);
    // (a) barriers
    printf(", \"barrier_cycles\": {");
    const int iters = 20000;
    bool first = true;
    for (int P : {32, 64, 128, 256, 512, 1024}) {
        bar_kernel<<<sms, P>>>(iters);
        CK(cudaDeviceSynchronize());
        bar_kernel<<<sms, P>>>(iters);
        CK(cudaMemcpyFromSymbol(h.data(), g_out, sizeof(long long) * sms));
        double m = 0;
        for (int i = 0; i < sms; ++i) m += (double)h[i] / iters;
        printf("%s\"%d\": %.2f", first ? "" : ", ", P, m / sms);
        first = false;
    }
    printf("}");
    // (b) flag ping-pong and atomics
    int* flags = nullptr;
    CK(cudaMalloc(&flags, 4096));
    for (int rep = 0; rep < 2; ++rep) {
        CK(cudaMemset(flags, 0, 4096));
        pingpong_kernel<<<2, 32>>>(flags, 20000);
        CK(cudaDeviceSynchronize());
    }
    CK(cudaMemcpyFromSymbol(h.data(), g_out, sizeof(long long)));
    printf(", \"flag_one_way_cycles\": %.1f", (double)h[0] / 20000 / 2);
    atomic_kernel<<<1, 32>>>(flags + 512, 20000);
    CK(cudaDeviceSynchronize());
    CK(cudaMemcpyFromSymbol(h.data(), g_out, sizeof(long long)));
    printf(", \"atomic_round_trip_cycles\": %.1f", (double)h[0] / 20000);
    atomic_kernel<<<sms, 32>>>(flags + 512, 2000);  // contended: every SM on one counter
    CK(cudaDeviceSynchronize());
    CK(cudaMemcpyFromSymbol(h.data(), g_out, sizeof(long long) * sms));
    {
        double m = 0;
        for (int i = 0; i < sms; ++i) m += (double)h[i] / 2000;
        printf(", \"atomic_round_trip_cycles_contended\": %.1f", m / sms);
    }
    // L: bulk TMA
    const size_t span = (size_t)2 << 30;
    uint8_t* src = nullptr;
    CK(cudaMalloc(&src, span));
    CK(cudaMemset(src, 1, span));
    CK(cudaFuncSetAttribute(tma_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 2 * 32768));
    printf(", \"tma\": [");
    first = true;
    // ctas per SM: 0 = one CTA on the whole GPU; k >= 1 = k CTAs on every SM (k double-buffered
    // copies in flight per SM: the kernels keep 16 warps x one prefetch in flight)
    for (uint32_t bytes : {1024u, 4096u, 6400u, 7168u, 16384u, 32768u}) {
        for (int k : {0, 1, 4, 8, 14}) {
            if (k * 2 * bytes > 220 * 1024) continue;
            const int grid = k ? sms * k : 1;
            const int chunks = k ? (int)(span / 4 / bytes / grid) : 2000;
            tma_kernel<<<grid, 32, 2 * bytes>>>(src, span, bytes, chunks);
            CK(cudaDeviceSynchronize());
            cudaEvent_t e0, e1;
            CK(cudaEventCreate(&e0));
            CK(cudaEventCreate(&e1));
            CK(cudaEventRecord(e0));
            tma_kernel<<<grid, 32, 2 * bytes>>>(src, span, bytes, chunks);
            CK(cudaEventRecord(e1));
            CK(cudaDeviceSynchronize());
            float ms = 0;
            CK(cudaEventElapsedTime(&ms, e0, e1));
            CK(cudaMemcpyFromSymbol(h.data(), g_out, sizeof(long long) * 4096));
            double cyc = 0;
            for (int i = 0; i < grid; ++i) cyc += (double)h[i];
            cyc /= grid;
            const double bytes_moved = (double)bytes * chunks;  // per CTA
            const double per_sm = k ? bytes_moved * k / cyc : bytes_moved / cyc;
            printf("%s{\"bytes\": %u, \"ctas\": %d, \"ctas_per_sm\": %d, \"bytes_per_clk_per_sm\": %.2f, "
                   "\"gb_per_s_total\": %.1f, \"mbar_wait_complete_cycles\": %lld}",
                   first ? "" : ", ", bytes, grid, k, per_sm, bytes_moved * grid / (ms * 1e-3) / 1e9, h[4095]);
            first = false;
        }
    }
    printf("]}\n");
    return 0;
}

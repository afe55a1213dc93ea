// probe.cu -- microbenchmarks of the roofline denominators of the pruning kernels
// (DESIGN.md "Rooflines"): the FP64 and FP32 FMA pipes and shared-memory load
// bandwidth of this GPU, measured with CUDA events (mpcgs_probe_peak, mpcgs.h).
// The pruning path is bound by the plain ALUs, so its roofline
// fraction needs these peaks measured rather than derived from unit counts.
#include <cuda_runtime.h>

#include "mpcgs.h"

namespace {

constexpr int PROBE_THREADS = 256;
constexpr int PROBE_CHAINS = 8;  // independent FMA chains per thread (covers the pipe latency)

template <typename T>
__global__ void __launch_bounds__(PROBE_THREADS) k_fma(T* out, int iters, T a, T b) {
    T x[PROBE_CHAINS];
#pragma unroll
    for (int k = 0; k < PROBE_CHAINS; ++k) x[k] = (T)(threadIdx.x + k) * (T)1e-3;
    for (int i = 0; i < iters; ++i) {
#pragma unroll
        for (int r = 0; r < 16; ++r)
#pragma unroll
            for (int k = 0; k < PROBE_CHAINS; ++k) x[k] = fma(x[k], a, b);
    }
    T s = 0;
#pragma unroll
    for (int k = 0; k < PROBE_CHAINS; ++k) s += x[k];
    if (s == (T)-1.2345) out[blockIdx.x] = s;  // keeps the chains live; never true
}

// ld.shared.v4.u32 (16 B per thread) over a 32 KB buffer, conflict-free addresses
__global__ void __launch_bounds__(PROBE_THREADS) k_lds(unsigned* out, int iters) {
    __shared__ __align__(16) unsigned buf[8192];
    for (int i = threadIdx.x; i < 8192; i += PROBE_THREADS) buf[i] = i * 2654435761u;
    __syncthreads();
    const unsigned base = (unsigned)__cvta_generic_to_shared(buf);
    unsigned acc = 0;
    unsigned off = (threadIdx.x * 16u) & 32767u;
    for (int i = 0; i < iters; ++i) {
#pragma unroll
        for (int r = 0; r < 8; ++r) {
            unsigned v0, v1, v2, v3;
            asm volatile("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];\n"
                         : "=r"(v0), "=r"(v1), "=r"(v2), "=r"(v3)
                         : "r"(base + ((off + r * 4096u) & 32767u)));
            acc ^= v0 ^ v1 ^ v2 ^ v3;
        }
        off = (off + 16u * PROBE_THREADS) & 32767u;
    }
    if (acc == 0x12345678u) out[blockIdx.x] = acc;
}

}  // namespace

extern "C" mpcgs_status mpcgs_probe_peak(int32_t kind, double* value) {
    if (!value || kind < 0 || kind > 2) return MPCGS_E_ARG;
    int dev = 0, sms = 0;
    if (cudaGetDevice(&dev) != cudaSuccess || cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess)
        return MPCGS_E_CUDA;
    void* out = nullptr;
    if (cudaMalloc(&out, 8 * 4096) != cudaSuccess) return MPCGS_E_NOMEM;
    cudaStream_t st;
    cudaEvent_t e0, e1;
    cudaStreamCreateWithFlags(&st, cudaStreamNonBlocking);
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    const int blocks = sms * 8;  // 2048 threads per SM
    const int iters = kind == 2 ? 4096 : 2048;
    auto launch = [&]() {
        if (kind == 0) k_fma<double><<<blocks, PROBE_THREADS, 0, st>>>((double*)out, iters, 1.0000001, 1e-9);
        else if (kind == 1) k_fma<float><<<blocks, PROBE_THREADS, 0, st>>>((float*)out, iters, 1.0000001f, 1e-9f);
        else k_lds<<<blocks, PROBE_THREADS, 0, st>>>((unsigned*)out, iters);
    };
    launch();  // warm-up (clocks up, module loaded)
    launch();
    float best = 1e30f;
    for (int r = 0; r < 5; ++r) {
        cudaEventRecord(e0, st);
        launch();
        cudaEventRecord(e1, st);
        cudaEventSynchronize(e1);
        float ms = 0.f;
        cudaEventElapsedTime(&ms, e0, e1);
        if (ms < best) best = ms;
    }
    const cudaError_t err = cudaGetLastError();
    cudaEventDestroy(e0);
    cudaEventDestroy(e1);
    cudaStreamDestroy(st);
    cudaFree(out);
    if (err != cudaSuccess) return MPCGS_E_CUDA;
    const double threads = (double)blocks * PROBE_THREADS;
    if (kind < 2)  // FMA = 2 flops
        *value = threads * iters * 16.0 * PROBE_CHAINS * 2.0 / (best * 1e-3) / 1e12;  // TFLOP/s
    else
        *value = threads * iters * 8.0 * 16.0 / (best * 1e-3) / 1e9;  // GB/s
    return MPCGS_OK;
}

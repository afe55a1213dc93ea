// step.cu -- one generalized Metropolis-Hastings step on the device
// (Alg. 1; Fig. 12), without host round trips:
//
//   k_context  (1 CTA)      target draw (4.3 L1079-1093, S7) and the shared
//                           neighbourhood context: feasible intervals, inactive
//                           lineage counts, closed-form transition weights and
//                           the backward messages P_i(n) (4.2 L986-1027, S9-S12)
//   k_propose  (1 warp/slot) forward walk + event placement (4.2 L1028-1043,
//                           S13-S15), tree patch, S_G (Eq. 18), Sethi-Ullman
//                           register schedule for the pruning kernel
//   k_draw     (1 CTA)      weights = softmax(logL) over N+1 states (Eq. 29-31,
//                           S18: the prior is recorded, never added), K inverse-
//                           CDF draws (L1140-1144), sample store, generator commit
#include <algorithm>
#include <cfloat>
#include <cstdio>

#include "step_body.cuh"

namespace mpcgs {

__global__ void __launch_bounds__(CTX_THREADS) k_context(DevState s, uint64_t seed, int64_t step_arg) {
    extern __shared__ __align__(16) double csm[];
    context_body<CTX_THREADS>(s, seed, step_arg, csm);
}

size_t context_smem_bytes(int n) {
    return sizeof(double) * ((size_t)(n - 1) + n + (n + 1) + (n + 2) + 6 * n + 3 * (n + 1)) +
           sizeof(int) * ((n + 1) + (2 * (size_t)n - 1) + 2 * (size_t)(n - 1)) + 16;
}

cudaError_t launch_context(const DevState& s, uint64_t seed, int64_t step, cudaStream_t st) {
    size_t smem = context_smem_bytes(s.n);
    static size_t attr_bytes = 48 * 1024;
    if (smem > attr_bytes) {
        cudaError_t e = cudaFuncSetAttribute(k_context, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        if (e != cudaSuccess) return e;
        attr_bytes = smem;
    }
    k_context<<<1, CTX_THREADS, smem, st>>>(s, seed, step);
    return cudaGetLastError();
}

template <typename E4, typename ET>
__global__ void __launch_bounds__(32) k_propose(DevState s, uint64_t seed, int64_t step_arg, int slot_first) {
    extern __shared__ __align__(16) int psm[];
    const int local = blockIdx.x;
    propose_warp<E4, ET>(s, seed, step_arg, slot_first + local, local, psm, s.sched_op + (size_t)local * s.nops,
                         reinterpret_cast<E4*>(s.sched_e) + (size_t)local * s.nops);
}

size_t propose_smem_bytes(int n) {
    const size_t nn = 2 * (size_t)n - 1;
    return sizeof(int) * (size_t)propose_int_words(n) + sizeof(double) * ((size_t)(n + 2) + (n + 1) + OM_STRIDE * (n + 1) + 2 * nn);
}

cudaError_t launch_propose(const DevState& s, uint64_t seed, int64_t step, int slot_first, int count,
                           cudaStream_t st) {
    if (count <= 0) return cudaSuccess;
    const size_t smem = propose_smem_bytes(s.n);
    static size_t attr64 = 48 * 1024, attr32 = 48 * 1024;
    if (s.precision == 32) {
        if (smem > attr32) {
            cudaError_t e = cudaFuncSetAttribute(k_propose<float4, float>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
            if (e != cudaSuccess) return e;
            attr32 = smem;
        }
        k_propose<float4, float><<<count, 32, smem, st>>>(s, seed, step, slot_first);
    } else {
        if (smem > attr64) {
            cudaError_t e = cudaFuncSetAttribute(k_propose<double4, double>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
            if (e != cudaSuccess) return e;
            attr64 = smem;
        }
        k_propose<double4, double><<<count, 32, smem, st>>>(s, seed, step, slot_first);
    }
    return cudaGetLastError();
}

template <int NT>
__global__ void __launch_bounds__(NT) k_draw(DevState s, uint64_t seed, int64_t step_arg, int N,
                                                       int K_arg, int burnin, int64_t M, int64_t total_steps) {
    extern __shared__ __align__(16) double dsm[];
    draw_body<NT>(s, seed, step_arg, N, K_arg, burnin, M, total_steps, dsm);
}

cudaError_t launch_draw(const DevState& s, uint64_t seed, int64_t step, int N, int K, int burnin, int64_t M,
                        int64_t total_steps, cudaStream_t st) {
    const size_t smem = std::max(3 * sizeof(double) * (size_t)(N + 1), context_smem_bytes(s.n));
    static size_t attr_bytes = 48 * 1024;
    if (smem > attr_bytes) {
        cudaError_t e = cudaFuncSetAttribute(k_draw<128>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        if (e == cudaSuccess)
            e = cudaFuncSetAttribute(k_draw<DRAW_THREADS>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        if (e != cudaSuccess) return e;
        attr_bytes = smem;
    }
    if (N <= 256) k_draw<128><<<1, 128, smem, st>>>(s, seed, step, N, K, burnin, M, total_steps);
    else k_draw<DRAW_THREADS><<<1, DRAW_THREADS, smem, st>>>(s, seed, step, N, K, burnin, M, total_steps);
    return cudaGetLastError();
}

}  // namespace mpcgs

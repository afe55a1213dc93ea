// theta.cu -- relative likelihood of theta over the sampled genealogies
// (Eq. 25-26; the paper's posterior likelihood kernel, 5.2.3
// L1417-1436).  By Eq. 18 a genealogy enters only through S_G, so
//   ln L(theta) = (n-1) ln(theta0/theta) + LSE_G[-S_G b] - ln M,  b = 1/theta - 1/theta0.
// The LSE shift is analytic (max_G -S_G b is attained at S_min or S_max), so a
// single pass suffices (the paper's max-reduction, L1425-1429, is not needed).
// All reductions run in a fixed order (deterministic results).
#include <cfloat>

#include "kernels.cuh"

namespace mpcgs {

constexpr int TH_THREADS = 256;

template <int NT>
__device__ double block_sum(double v, double* s_red) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_down_sync(0xffffffffu, v, o);
    if ((threadIdx.x & 31) == 0) s_red[threadIdx.x >> 5] = v;
    __syncthreads();
    double t = 0.0;
    if (threadIdx.x == 0)
        for (int w = 0; w < NT / 32; ++w) t += s_red[w];
    __syncthreads();
    return t;  // valid in thread 0
}

__global__ void __launch_bounds__(1024) k_minmax(const double* __restrict__ S, int64_t M, double* out2) {
    __shared__ double smin[32], smax[32];
    double lo = CUDART_INF, hi = -CUDART_INF;
    for (int64_t i = threadIdx.x; i < M; i += blockDim.x) {
        const double v = S[i];
        lo = fmin(lo, v);
        hi = fmax(hi, v);
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        lo = fmin(lo, __shfl_xor_sync(0xffffffffu, lo, o));
        hi = fmax(hi, __shfl_xor_sync(0xffffffffu, hi, o));
    }
    if ((threadIdx.x & 31) == 0) {
        smin[threadIdx.x >> 5] = lo;
        smax[threadIdx.x >> 5] = hi;
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        for (int w = 1; w < (int)(blockDim.x >> 5); ++w) {
            lo = fmin(lo, smin[w]);
            hi = fmax(hi, smax[w]);
        }
        lo = fmin(lo, smin[0]);
        hi = fmax(hi, smax[0]);
        out2[0] = lo;
        out2[1] = hi;
    }
}

// One CTA per grid point g: theta_g log-spaced over [lo, hi].
__global__ void __launch_bounds__(TH_THREADS) k_theta_grid(const double* __restrict__ S, int64_t M, int n,
                                                          double theta0, double lo, double hi, int G,
                                                          double smin, double smax, double* out) {
    __shared__ double s_red[TH_THREADS / 32];
    const int g = blockIdx.x;
    const double theta = exp(log(lo) + (log(hi) - log(lo)) * (double)g / (double)(G - 1));
    const double b = 1.0 / theta - 1.0 / theta0;
    const double shift = b > 0.0 ? -smin * b : -smax * b;
    double acc = 0.0;
    for (int64_t i = threadIdx.x; i < M; i += TH_THREADS) acc += exp(-S[i] * b - shift);
    const double tot = block_sum<TH_THREADS>(acc, s_red);
    if (threadIdx.x == 0) {
        out[g] = theta;
        out[G + g] = (double)(n - 1) * log(theta0 / theta) + shift + log(tot) - log((double)M);
    }
}

// Weighted moments at one theta about `center`: sum w, sum w (S-c), sum w (S-c)^2
// with w = exp(-S b - shift).  Multi-CTA; the last CTA reduces in CTA order.
__global__ void __launch_bounds__(TH_THREADS) k_theta_moments(const double* __restrict__ S, int64_t M,
                                                             double theta0, double theta, double shift,
                                                             double center, double* part, unsigned* cnt,
                                                             double* out3) {
    __shared__ double s_red[TH_THREADS / 32];
    __shared__ bool s_last;
    const double b = 1.0 / theta - 1.0 / theta0;
    double w0 = 0.0, w1 = 0.0, w2 = 0.0;
    for (int64_t i = (int64_t)blockIdx.x * TH_THREADS + threadIdx.x; i < M; i += (int64_t)gridDim.x * TH_THREADS) {
        const double sv = S[i];
        const double w = exp(-sv * b - shift);
        const double d = sv - center;
        w0 += w;
        w1 += w * d;
        w2 += w * d * d;
    }
    w0 = block_sum<TH_THREADS>(w0, s_red);
    w1 = block_sum<TH_THREADS>(w1, s_red);
    w2 = block_sum<TH_THREADS>(w2, s_red);
    if (threadIdx.x == 0) {
        part[3 * blockIdx.x + 0] = w0;
        part[3 * blockIdx.x + 1] = w1;
        part[3 * blockIdx.x + 2] = w2;
        __threadfence();
        s_last = atomicAdd(cnt, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (s_last && threadIdx.x == 0) {
        __threadfence();
        const volatile double* p = part;
        double t0 = 0.0, t1 = 0.0, t2 = 0.0;
        for (unsigned k = 0; k < gridDim.x; ++k) {
            t0 += p[3 * k + 0];
            t1 += p[3 * k + 1];
            t2 += p[3 * k + 2];
        }
        out3[0] = t0;
        out3[1] = t1;
        out3[2] = t2;
        *cnt = 0u;
    }
}

cudaError_t launch_minmax(const double* S, int64_t M, double* out2, cudaStream_t st) {
    k_minmax<<<1, 1024, 0, st>>>(S, M, out2);
    return cudaGetLastError();
}

cudaError_t launch_theta_grid(const double* S, int64_t M, int n, double theta0, double lo, double hi, int G,
                              double smin, double smax, double* out, cudaStream_t st) {
    k_theta_grid<<<G, TH_THREADS, 0, st>>>(S, M, n, theta0, lo, hi, G, smin, smax, out);
    return cudaGetLastError();
}

cudaError_t launch_theta_moments(const double* S, int64_t M, double theta0, double theta, double shift,
                                 double center, double* part, unsigned* cnt, double* out3, cudaStream_t st) {
    int blocks = (int)((M + TH_THREADS - 1) / TH_THREADS);
    if (blocks > 296) blocks = 296;  // 2 per SM on 148 SMs
    if (blocks < 1) blocks = 1;
    k_theta_moments<<<blocks, TH_THREADS, 0, st>>>(S, M, theta0, theta, shift, center, part, cnt, out3);
    return cudaGetLastError();
}

}  // namespace mpcgs

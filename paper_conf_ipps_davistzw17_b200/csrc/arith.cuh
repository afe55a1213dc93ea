// arith.cuh -- per-node F81 pruning arithmetic shared by the pruning kernels
// (prune.cu) and the incremental rescoring kernels (incr.cu).  Eq. 19-20 with
// exact power-of-two underflow rescaling (S5).
#pragma once
#include "common.cuh"

namespace mpcgs {

template <typename T>
struct Traits;
template <>
struct Traits<double> {
    using E4 = double4;
    // rescale when max < 2^-256: hi word of the IEEE double < (1023-256) << 20
    static constexpr int TS = 256;
};
template <>
struct Traits<float> {
    using E4 = float4;
    static constexpr int TS = 32;  // products of two 2^-32-bounded vectors stay normal (S5)
};

__device__ __forceinline__ int hi_bits(double x) { return __double2hiint(x); }
__device__ __forceinline__ int hi_bits(float x) { return __float_as_int(x); }

// Rescale v by 2^k so that max(v) lands in [1, 2) when max(v) < 2^-TS; scale -= k.
__device__ __forceinline__ void maybe_rescale(double (&v)[4], int& scale) {
    int m = max(max(hi_bits(v[0]), hi_bits(v[1])), max(hi_bits(v[2]), hi_bits(v[3])));
    if (m < ((1023 - Traits<double>::TS) << 20)) {
        int k = 1023 - (m >> 20);                       // max * 2^k in [1, 2) (normal max)
        k = min(k, 1000);
        double f = __hiloint2double((1023 + k) << 20, 0);
        v[0] *= f; v[1] *= f; v[2] *= f; v[3] *= f;
        scale += k;
    }
}
__device__ __forceinline__ void maybe_rescale(float (&v)[4], int& scale) {
    int m = max(max(hi_bits(v[0]), hi_bits(v[1])), max(hi_bits(v[2]), hi_bits(v[3])));
    if (m < ((127 - Traits<float>::TS) << 23)) {
        int k = 127 - (m >> 23);
        k = min(k, 120);
        float f = __int_as_float((127 + k) << 23);
        v[0] *= f; v[1] *= f; v[2] *= f; v[3] *= f;
        scale += k;
    }
}

// branch(L)_X = sum_Y P_XY(t) L_Y = e L_X + em (pi . L)   (Eq. 19 + Eq. 20)
template <typename T>
__device__ __forceinline__ void branch(T (&r)[4], T e, T em, const T (&pi)[4]) {
    // sequential pi . L (fewest FP instructions; four sites per thread supply the ILP)
    T s = pi[0] * r[0];
    s = fma(pi[1], r[1], s);
    s = fma(pi[2], r[2], s);
    s = fma(pi[3], r[3], s);
    const T t = em * s;
    r[0] = fma(e, r[0], t);
    r[1] = fma(e, r[1], t);
    r[2] = fma(e, r[2], t);
    r[3] = fma(e, r[3], t);
}

// tip(x)_X = P_{X,x}(t) = e [X==x] + em pi_x   (tips are indicators, L673-676)
template <typename T>
__device__ __forceinline__ void tipvec(T (&r)[4], int x, T e, T em, const T (&pi)[4]) {
    T px = x == 0 ? pi[0] : (x == 1 ? pi[1] : (x == 2 ? pi[2] : pi[3]));
    T c = em * px;
    T ce = c + e;
    r[0] = x == 0 ? ce : c;
    r[1] = x == 1 ? ce : c;
    r[2] = x == 2 ? ce : c;
    r[3] = x == 3 ? ce : c;
}

template <typename T>
__device__ __forceinline__ void ld4(T (&r)[4], const T* p);
template <>
__device__ __forceinline__ void ld4<double>(double (&r)[4], const double* p) {
    const double2 a = reinterpret_cast<const double2*>(p)[0];
    const double2 b = reinterpret_cast<const double2*>(p)[1];
    r[0] = a.x; r[1] = a.y; r[2] = b.x; r[3] = b.y;
}
template <>
__device__ __forceinline__ void ld4<float>(float (&r)[4], const float* p) {
    const float4 a = *reinterpret_cast<const float4*>(p);
    r[0] = a.x; r[1] = a.y; r[2] = a.z; r[3] = a.w;
}

template <typename T>
__device__ __forceinline__ void st4(T* p, const T (&r)[4]);
template <>
__device__ __forceinline__ void st4<double>(double* p, const double (&r)[4]) {
    reinterpret_cast<double2*>(p)[0] = make_double2(r[0], r[1]);
    reinterpret_cast<double2*>(p)[1] = make_double2(r[2], r[3]);
}
template <>
__device__ __forceinline__ void st4<float>(float* p, const float (&r)[4]) {
    *reinterpret_cast<float4*>(p) = make_float4(r[0], r[1], r[2], r[3]);
}

template <typename T>
__device__ __forceinline__ T pick4(const T (&v)[4], int x) {
    return x == 0 ? v[0] : (x == 1 ? v[1] : (x == 2 ? v[2] : v[3]));
}

// exponent test of one 4-vector: k > 0 if max < 2^-TS (then max * 2^k in [1, 2))
__device__ __forceinline__ int rescale_k(const double (&r)[4]) {
    const int m = max(max(hi_bits(r[0]), hi_bits(r[1])), max(hi_bits(r[2]), hi_bits(r[3])));
    return m < ((1023 - Traits<double>::TS) << 20) ? min(1023 - (m >> 20), 1000) : 0;
}
__device__ __forceinline__ int rescale_k(const float (&r)[4]) {
    const int m = max(max(hi_bits(r[0]), hi_bits(r[1])), max(hi_bits(r[2]), hi_bits(r[3])));
    return m < ((127 - Traits<float>::TS) << 23) ? min(127 - (m >> 23), 120) : 0;
}
__device__ __forceinline__ double pow2(int k, double) { return __hiloint2double((1023 + k) << 20, 0); }
__device__ __forceinline__ float pow2(int k, float) { return __int_as_float((127 + k) << 23); }

// Rescale when any site of any lane has max < 2^-TS: the per-site test is
// cheap (integer max of the high words); the multiply is a rare warp-uniform branch.
__device__ __forceinline__ bool small4(const double (&r)[4]) {
    const int m = max(max(hi_bits(r[0]), hi_bits(r[1])), max(hi_bits(r[2]), hi_bits(r[3])));
    return m < ((1023 - Traits<double>::TS) << 20);
}
__device__ __forceinline__ bool small4(const float (&r)[4]) {
    const int m = max(max(hi_bits(r[0]), hi_bits(r[1])), max(hi_bits(r[2]), hi_bits(r[3])));
    return m < ((127 - Traits<float>::TS) << 23);
}
// Accumulator of site log-likelihoods (Eq. 22 read as a product over sites, S4):
// a product kept as mantissa * 2^expo (one log at the end), or -- when the
// sites are compressed patterns -- a sum of count * ln L_s.
// `scale` is the power-of-two exponent removed from the site's vectors.
template <bool W>  // W: compressed sites with weights (separate instantiation: keeps the log out of the hot loop)
struct SiteAcc {
    double mant = 1.0, wlog = 0.0;
    int expo = 0;
    __device__ __forceinline__ void add(double ls, int scale, const double* __restrict__ w, int site) {
        if constexpr (W) {
            wlog += w[site] * (log(ls) - (double)scale * 0.69314718055994530942);
        } else {
            mant *= ls;
            const int hi = __double2hiint(mant);
            const int ex = ((hi >> 20) & 2047) - 1023;
            if (ex > -1023) {  // normal: move the exponent into expo, mantissa to [1, 2)
                mant = __hiloint2double((hi & 0x800FFFFF) | (1023 << 20), __double2loint(mant));
                expo += ex;
            }
            expo -= scale;
        }
    }
    __device__ __forceinline__ double total() const {
        if constexpr (W) return wlog;
        return mant > 0.0 ? log(mant) + (double)expo * 0.69314718055994530942 : -INFINITY;
    }
};

}  // namespace mpcgs

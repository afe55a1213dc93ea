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

// The same branch divided by e (a per-branch constant, the same at every site):
// branch(L)_X / e = L_X + r (pi . L), r = em / e = e^{ut} - 1.  One FP instruction
// per site fewer than branch(); the table kernel adds sum ln e per site back once
// per genealogy (prune_kernels.cuh, unit_branch).
template <typename T>
__device__ __forceinline__ void branch_unit(T (&v)[4], T r, const T (&pi)[4]) {
    T s = pi[0] * v[0];
    s = fma(pi[1], v[1], s);
    s = fma(pi[2], v[2], s);
    s = fma(pi[3], v[3], s);
    v[0] = fma(r, s, v[0]);
    v[1] = fma(r, s, v[1]);
    v[2] = fma(r, s, v[2]);
    v[3] = fma(r, s, v[3]);
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
    __device__ __forceinline__ void reset() {
        mant = 1.0;
        wlog = 0.0;
        expo = 0;
    }
};

// ---------------------------------------------------------------------------
// Exact site sums (P22: the same logL for every tiling and world size).
// A genealogy's ln P(D|G) (Eq. 22 read as a product, S4) is the sum of per-unit
// terms: a unit is a fixed range of sites (a function of n, L and the precision
// only), within which each thread multiplies its own sites' likelihoods and
// takes one log.  Those terms are added as 128-bit two's-complement fixed point
// with 64 fraction bits, i.e. as integers: associative, so the order in which
// threads, CTAs and tiles add them (and hence the pruning tiling, which follows
// the number of proposals a rank scores) cannot change the result.  Each term
// is truncated to a multiple of 2^-64 (error < 5.5e-20 per term); the sum is
// rounded to double once at the end.  A zero site likelihood makes the total
// -inf (S6); |term| must stay below 2^62.
// ---------------------------------------------------------------------------
struct Exact128 {
    unsigned long long lo = 0ull;
    long long hi = 0ll;
    unsigned flags = 0u;  // bit 0: -inf (a zero likelihood), bit 1: NaN / out of range

    __device__ __forceinline__ void add_fixed(unsigned long long ql, long long qh) {
        const unsigned long long nl = lo + ql;
        hi += qh + (long long)(nl < lo);
        lo = nl;
    }
    __device__ __forceinline__ void add(double v) {
        if (v == 0.0) return;
        if (!(v > -INFINITY)) {
            flags |= (v == -INFINITY) ? 1u : 2u;
            return;
        }
        const unsigned long long bits = (unsigned long long)__double_as_longlong(v);
        int e = (int)((bits >> 52) & 0x7FFull);
        unsigned long long m = bits & 0xFFFFFFFFFFFFFull;
        if (e == 0x7FF) {  // +inf
            flags |= 2u;
            return;
        }
        if (e == 0) e = 1;                 // subnormal
        else m |= 1ull << 52;
        const int sh = e - 1075 + 64;      // |v| 2^64 = m 2^sh
        unsigned long long ql, qh;
        if (sh >= 74) {                    // |v| >= 2^62: outside the accumulator's range
            flags |= 2u;
            return;
        } else if (sh >= 64) {
            qh = m << (sh - 64);
            ql = 0ull;
        } else if (sh > 0) {
            ql = m << sh;
            qh = m >> (64 - sh);
        } else if (sh > -64) {
            ql = m >> (-sh);
            qh = 0ull;
        } else {
            return;                        // below 2^-64
        }
        if (bits >> 63) {                  // negate (two's complement)
            ql = ~ql + 1ull;
            qh = ~qh + (unsigned long long)(ql == 0ull);
        }
        add_fixed(ql, (long long)qh);
    }
    __device__ __forceinline__ void add(const Exact128& o) {
        add_fixed(o.lo, o.hi);
        flags |= o.flags;
    }
    __device__ __forceinline__ void shfl_down_add(int off) {
        Exact128 o;
        o.lo = __shfl_down_sync(0xffffffffu, lo, off);
        o.hi = __shfl_down_sync(0xffffffffu, hi, off);
        o.flags = __shfl_down_sync(0xffffffffu, flags, off);
        add(o);
    }
};

__device__ __forceinline__ double exact_to_double(unsigned long long lo, long long hi, unsigned flags) {
    if (flags & 2u) return __longlong_as_double(0x7FF8000000000000ll);  // NaN
    if (flags & 1u) return -INFINITY;
    return (double)hi + (double)lo * 5.421010862427522e-20;          // hi + lo 2^-64
}

template <int NT>
struct ExactScratch {
    unsigned long long w[3 * (NT / 32) + 1];
};

// Per-genealogy accumulator in device memory: [0] lo, [1] hi, [2] flags (zero on entry;
// reset by the CTA that completes the genealogy).
// Block-reduce v (exactly), add it to acc with 64-bit atomics (carry from the low
// word's old value), and let the last of `tiles` CTAs write the double (+ add) to *out.
// scratch: shared memory of >= 3 * NT / 32 + 1 words, free for the call (the table
// kernel passes its tip-code staging buffers, so the commit adds no static shared
// memory that would cost it a fused triplet table).
template <int NT>
__device__ __forceinline__ void exact_commit(Exact128 v, unsigned long long* acc, unsigned* cnt, int tiles,
                                             double* out, unsigned long long* scratch, double add = 0.0) {
    unsigned long long* s_lo = scratch;
    long long* s_hi = reinterpret_cast<long long*>(scratch + NT / 32);
    unsigned long long* s_fl = scratch + 2 * (NT / 32);
    volatile unsigned long long* s_last = scratch + 3 * (NT / 32);
    const int tid = threadIdx.x;
#pragma unroll
    for (int off = 16; off > 0; off >>= 1) v.shfl_down_add(off);
    if ((tid & 31) == 0) {
        s_lo[tid >> 5] = v.lo;
        s_hi[tid >> 5] = v.hi;
        s_fl[tid >> 5] = v.flags;
    }
    __syncthreads();
    if (tid == 0) {
        Exact128 t;
        for (int w = 0; w < NT / 32; ++w) {
            Exact128 o;
            o.lo = s_lo[w];
            o.hi = s_hi[w];
            o.flags = (unsigned)s_fl[w];
            t.add(o);
        }
        const unsigned long long old = atomicAdd(acc, t.lo);
        const unsigned long long carry = (old + t.lo < old) ? 1ull : 0ull;
        atomicAdd(acc + 1, (unsigned long long)t.hi + carry);
        if (t.flags) atomicOr(acc + 2, (unsigned long long)t.flags);
        __threadfence();
        const unsigned prev = atomicAdd(cnt, 1u);
        *s_last = (prev == (unsigned)(tiles - 1)) ? 1ull : 0ull;
    }
    __syncthreads();
    if (*s_last && tid == 0) {
        __threadfence();
        const volatile unsigned long long* va = acc;
        const unsigned long long lo = va[0], hi = va[1], fl = va[2];
        *out = exact_to_double(lo, (long long)hi, (unsigned)fl) + add;  // add: the same in every CTA of the tree
        acc[0] = 0ull;
        acc[1] = 0ull;
        acc[2] = 0ull;
        *cnt = 0u;
    }
    __syncthreads();
}

}  // namespace mpcgs

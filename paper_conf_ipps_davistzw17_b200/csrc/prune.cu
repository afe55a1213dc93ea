// prune.cu -- Felsenstein pruning data likelihood (Eq. 19-22) of many
// genealogies over all sites, F81 closed form (Eq. 20), on the CUDA cores.
//
// Grid: (site tiles, trees).  One CTA = one tree x one tile of sites; each
// thread owns sites tid, tid+blockDim, ... of the tile.  The tree's post-order
// schedule (common.cuh) is staged in shared memory once per CTA and read as
// warp-uniform broadcasts; the live partial likelihood vectors of a site sit in
// a register stack R[D][4] addressed only with compile-time indices (the switch
// below dispatches on the uniform (type, sp) code), so no partial ever touches
// shared or global memory.  Underflow: after each node the vector is rescaled
// by an exact power of two when its max drops below 2^-TS (S5), with one
// integer exponent per site.  Per-site likelihoods (Eq. 21) are multiplied
// into a mantissa/exponent accumulator, so each thread takes one log at the
// end (Eq. 22 read as a product over sites, S4).  CTA sums are reduced in a
// fixed order by the last CTA of each tree (deterministic, P22).
#include "common.cuh"
#include "kernels.cuh"

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
    T s = pi[0] * r[0];
    s = fma(pi[1], r[1], s);
    s = fma(pi[2], r[2], s);
    s = fma(pi[3], r[3], s);
    T t = em * s;
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

template <typename T, int D, int S>
__device__ __forceinline__ void op_tt(T (&R)[D][4], uint32_t code, const typename Traits<T>::E4& ed,
                                      const uint8_t* __restrict__ codes, int Lpad, int site,
                                      const T (&pi)[4], int& scale) {
    if constexpr (S < D) {
        int ta = (code >> 6) & 2047, tb = (code >> 17) & 2047;
        int xa = __ldg(codes + (size_t)ta * Lpad + site);
        int xb = __ldg(codes + (size_t)tb * Lpad + site);
        T va[4], vb[4];
        tipvec<T>(va, xa, ed.x, ed.y, pi);
        tipvec<T>(vb, xb, ed.z, ed.w, pi);
#pragma unroll
        for (int i = 0; i < 4; ++i) R[S][i] = va[i] * vb[i];
        maybe_rescale(R[S], scale);
    }
}

template <typename T, int D, int S>
__device__ __forceinline__ void op_ts(T (&R)[D][4], uint32_t code, const typename Traits<T>::E4& ed,
                                      const uint8_t* __restrict__ codes, int Lpad, int site,
                                      const T (&pi)[4], int& scale) {
    if constexpr (S >= 1 && S <= D) {
        int ta = (code >> 6) & 2047;
        int xa = __ldg(codes + (size_t)ta * Lpad + site);
        T va[4];
        tipvec<T>(va, xa, ed.x, ed.y, pi);
        branch<T>(R[S - 1], ed.z, ed.w, pi);
#pragma unroll
        for (int i = 0; i < 4; ++i) R[S - 1][i] *= va[i];
        maybe_rescale(R[S - 1], scale);
    }
}

template <typename T, int D, int S>
__device__ __forceinline__ void op_ss(T (&R)[D][4], const typename Traits<T>::E4& ed, const T (&pi)[4],
                                      int& scale) {
    if constexpr (S >= 2 && S <= D) {
        branch<T>(R[S - 2], ed.x, ed.y, pi);
        branch<T>(R[S - 1], ed.z, ed.w, pi);
#pragma unroll
        for (int i = 0; i < 4; ++i) R[S - 2][i] *= R[S - 1][i];
        maybe_rescale(R[S - 2], scale);
    }
}

#define MPCGS_OPCASE(S)                                                                     \
    case (OP_TT | ((S) << 2)): op_tt<T, D, S>(R, code, ed, codes, Lpad, site, pi, scale); break; \
    case (OP_TS | ((S) << 2)): op_ts<T, D, S>(R, code, ed, codes, Lpad, site, pi, scale); break; \
    case (OP_SS | ((S) << 2)): op_ss<T, D, S>(R, ed, pi, scale); break;

template <typename T, int D>
__global__ void __launch_bounds__(PRUNE_THREADS) k_prune(PruneArgs a) {
    using E4 = typename Traits<T>::E4;
    extern __shared__ __align__(16) unsigned char smem_raw[];
    E4* s_e = reinterpret_cast<E4*>(smem_raw);
    uint32_t* s_op = reinterpret_cast<uint32_t*>(smem_raw + sizeof(E4) * a.nops);
    __shared__ double s_red[PRUNE_THREADS / 32];
    __shared__ bool s_last;

    const int tree = blockIdx.y;
    const int tile = blockIdx.x;
    const uint32_t* __restrict__ gop = a.sched_op + (size_t)tree * a.nops;
    const E4* __restrict__ ge = reinterpret_cast<const E4*>(a.sched_e) + (size_t)tree * a.nops;
    for (int i = threadIdx.x; i < a.nops; i += blockDim.x) {
        s_op[i] = gop[i];
        s_e[i] = ge[i];
    }
    __syncthreads();

    const T pi[4] = {(T)a.pi[0], (T)a.pi[1], (T)a.pi[2], (T)a.pi[3]};
    const uint8_t* __restrict__ codes = a.codes;
    const int Lpad = a.Lpad;
    const int s_begin = tile * a.sites_per_cta;
    const int s_end = min(a.L, s_begin + a.sites_per_cta);

    double mant = 1.0;  // product of site likelihoods = mant * 2^expo
    int expo = 0;
    T R[D][4];
#pragma unroll
    for (int i = 0; i < D; ++i)
#pragma unroll
        for (int j = 0; j < 4; ++j) R[i][j] = T(0);

    for (int site = s_begin + threadIdx.x; site < s_end; site += blockDim.x) {
        int scale = 0;
        for (int op = 0; op < a.nops; ++op) {
            const uint32_t code = s_op[op];
            const E4 ed = s_e[op];
            switch (code & 63u) {
                MPCGS_OPCASE(0) MPCGS_OPCASE(1) MPCGS_OPCASE(2) MPCGS_OPCASE(3) MPCGS_OPCASE(4)
                MPCGS_OPCASE(5) MPCGS_OPCASE(6) MPCGS_OPCASE(7) MPCGS_OPCASE(8) MPCGS_OPCASE(9)
                MPCGS_OPCASE(10) MPCGS_OPCASE(11)
                default: break;
            }
        }
        // Eq. 21: L_s = sum_X pi_X L_root(X), root partial in R[0]
        T ls = pi[0] * R[0][0];
        ls = fma(pi[1], R[0][1], ls);
        ls = fma(pi[2], R[0][2], ls);
        ls = fma(pi[3], R[0][3], ls);
        mant *= (double)ls;
        int hi = __double2hiint(mant);
        int ex = ((hi >> 20) & 2047) - 1023;
        if (ex > -1023) {  // normal: move the exponent into expo, mantissa to [1, 2)
            mant = __hiloint2double((hi & 0x800FFFFF) | (1023 << 20), __double2loint(mant));
            expo += ex;
        }
        expo -= scale;
    }
    // ln of this thread's product; -inf if any site likelihood was 0 (S6)
    double ll = (mant > 0.0) ? log(mant) + (double)expo * 0.69314718055994530942 : -INFINITY;
    if (s_begin + (int)threadIdx.x >= s_end) ll = 0.0;

    // block reduction in a fixed order
#pragma unroll
    for (int off = 16; off > 0; off >>= 1) ll += __shfl_down_sync(0xffffffffu, ll, off);
    if ((threadIdx.x & 31) == 0) s_red[threadIdx.x >> 5] = ll;
    __syncthreads();
    if (threadIdx.x == 0) {
        double t = 0.0;
        for (int w = 0; w < (int)(blockDim.x >> 5); ++w) t += s_red[w];
        a.tile_part[(size_t)tree * a.tiles + tile] = t;
        __threadfence();
        unsigned prev = atomicAdd(a.tile_cnt + tree, 1u);
        s_last = (prev == (unsigned)(a.tiles - 1));
    }
    __syncthreads();
    if (s_last && threadIdx.x == 0) {
        __threadfence();
        double t = 0.0;
        const volatile double* tp = a.tile_part + (size_t)tree * a.tiles;
        for (int k = 0; k < a.tiles; ++k) t += tp[k];
        a.out[(size_t)(a.out_first + tree) * a.out_stride] = t;
        a.tile_cnt[tree] = 0u;
    }
}

template <typename T, int D>
static cudaError_t launch_one(const PruneArgs& a, int ntrees, cudaStream_t st) {
    size_t smem = (size_t)a.nops * (sizeof(typename Traits<T>::E4) + sizeof(uint32_t));
    auto kern = k_prune<T, D>;
    static size_t attr_bytes = 48 * 1024;  // raised once, outside graph capture (first launch is at init)
    if (smem > attr_bytes) {
        cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        if (e != cudaSuccess) return e;
        attr_bytes = smem;
    }
    dim3 grid(a.tiles, ntrees);
    kern<<<grid, PRUNE_THREADS, smem, st>>>(a);
    return cudaGetLastError();
}

int prune_depth_for(int n) {
    int d = 0;
    while ((2 << d) <= n) ++d;  // floor(log2 n) = max Sethi-Ullman need of an n-tip tree
    if (d <= 4) return 4;
    if (d <= 6) return 6;
    if (d <= 8) return 8;
    return 10;
}

cudaError_t launch_prune(const PruneArgs& a, int ntrees, int depth, int precision, cudaStream_t st) {
    if (ntrees <= 0) return cudaSuccess;
    if (precision == 32) {
        switch (depth) {
            case 4: return launch_one<float, 4>(a, ntrees, st);
            case 6: return launch_one<float, 6>(a, ntrees, st);
            case 8: return launch_one<float, 8>(a, ntrees, st);
            default: return launch_one<float, 10>(a, ntrees, st);
        }
    }
    switch (depth) {
        case 4: return launch_one<double, 4>(a, ntrees, st);
        case 6: return launch_one<double, 6>(a, ntrees, st);
        case 8: return launch_one<double, 8>(a, ntrees, st);
        default: return launch_one<double, 10>(a, ntrees, st);
    }
}

}  // namespace mpcgs

// prune_kernels.cuh -- Felsenstein pruning data likelihood (Eq. 19-22) of many
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
#pragma once
#include <algorithm>
#include <cstdio>
#include <type_traits>

#include "arith.cuh"
#include "common.cuh"
#include "kernels.cuh"

namespace mpcgs {

// tip vector of an F81 tip child: base x (0..3), or base-set mask x (AMB, S24):
// v_X = e [X in set] + em pi(set)
template <typename T, bool AMB>
__device__ __forceinline__ void tip81(T (&r)[4], int x, T e, T em, const T (&pi)[4]) {
    if constexpr (AMB) {
        const T ps = ((x & 1) ? pi[0] : T(0)) + ((x & 2) ? pi[1] : T(0)) + ((x & 4) ? pi[2] : T(0)) +
                     ((x & 8) ? pi[3] : T(0));
        const T c = em * ps;
#pragma unroll
        for (int i = 0; i < 4; ++i) r[i] = ((x >> i) & 1) ? c + e : c;
    } else {
        tipvec<T>(r, x, e, em, pi);
    }
}

template <typename T, int D, int S, bool AMB>
__device__ __forceinline__ void op_tt(T (&R)[D][4], uint32_t code, const typename Traits<T>::E4& ed,
                                      const uint8_t* __restrict__ codes, int Lpad, int site,
                                      const T (&pi)[4], int& scale) {
    if constexpr (S < D) {
        int ta = (code >> 6) & 2047, tb = (code >> 17) & 2047;
        int xa = __ldg(codes + (size_t)ta * Lpad + site);
        int xb = __ldg(codes + (size_t)tb * Lpad + site);
        T va[4], vb[4];
        tip81<T, AMB>(va, xa, ed.x, ed.y, pi);
        tip81<T, AMB>(vb, xb, ed.z, ed.w, pi);
#pragma unroll
        for (int i = 0; i < 4; ++i) R[S][i] = va[i] * vb[i];
        maybe_rescale(R[S], scale);
    }
}

template <typename T, int D, int S, bool AMB>
__device__ __forceinline__ void op_ts(T (&R)[D][4], uint32_t code, const typename Traits<T>::E4& ed,
                                      const uint8_t* __restrict__ codes, int Lpad, int site,
                                      const T (&pi)[4], int& scale) {
    if constexpr (S >= 1 && S <= D) {
        int ta = (code >> 6) & 2047;
        int xa = __ldg(codes + (size_t)ta * Lpad + site);
        T va[4];
        tip81<T, AMB>(va, xa, ed.x, ed.y, pi);
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

// ---- general reversible model: per-op P matrices {P_a, P_b}
// (row-major, row = parent state) formed by k_pmat; the tip vector of state x is
// column x of P (Eq. 19 with a one-hot child partial), a branch is P . R.
template <typename T, bool AMB>
__device__ __forceinline__ void gm_tip(T (&v)[4], const T* __restrict__ P, int x) {
    if constexpr (AMB) {  // base-set mask: sum of the set's columns (S24)
#pragma unroll
        for (int i = 0; i < 4; ++i)
            v[i] = ((x & 1) ? __ldg(P + i * 4) : T(0)) + ((x & 2) ? __ldg(P + i * 4 + 1) : T(0)) +
                   ((x & 4) ? __ldg(P + i * 4 + 2) : T(0)) + ((x & 8) ? __ldg(P + i * 4 + 3) : T(0));
    } else {
#pragma unroll
        for (int i = 0; i < 4; ++i) v[i] = __ldg(P + i * 4 + x);
    }
}

template <typename T>
__device__ __forceinline__ void gm_branch(T (&R)[4], const T* __restrict__ P) {
    T o[4];
#pragma unroll
    for (int i = 0; i < 4; ++i) {
        T v = P[i * 4] * R[0];
        v = fma(P[i * 4 + 1], R[1], v);
        v = fma(P[i * 4 + 2], R[2], v);
        o[i] = fma(P[i * 4 + 3], R[3], v);
    }
#pragma unroll
    for (int i = 0; i < 4; ++i) R[i] = o[i];
}

// ---- structured F84 / HKY85 branches (table kernel; host.cu model_consts): a branch
// of length t is the record C = {a, b_R, b_Y, c_R, c_Y} with
//   (P(t) v)_i = a T + b_g G_g + c_g v_i,   T = pi . v,  G_g = sum_{j in g} pi_j v_j,
// a = 1 - e^{-s t}, b_g = (e^{-s t} - e^{-s A_g t}) / Pi_g, c_g = e^{-s A_g t}; purines A, G
// (0, 2), pyrimidines C, T (1, 3).  12 FP instructions per branch instead of the 16 of a
// 4x4 matrix-vector product, and 5 values per branch instead of 16.
constexpr int GMC = 8;  // doubles / floats per branch record (5 used, padded for alignment)
template <typename T>
__device__ __forceinline__ void gm_coef(const double* __restrict__ mc, double t, T* C) {
    const double s = mc[0];
    const double e1m = -expm1(-s * t);  // 1 - e^{-s t}
    const double e1 = exp(-s * t);
    C[0] = (T)e1m;
#pragma unroll
    for (int g = 0; g < 2; ++g) {
        const double A = mc[1 + g], Pi = mc[3 + g];
        const double eg = exp(-s * A * t);
        // e^{-s t} - e^{-s A t} without cancellation
        const double d = A >= 1.0 ? e1 * -expm1(-s * (A - 1.0) * t) : -eg * -expm1(-s * (1.0 - A) * t);
        C[1 + g] = (T)(d / Pi);
        C[3 + g] = (T)eg;
    }
#pragma unroll
    for (int k = 5; k < GMC; ++k) C[k] = T(0);
}
template <typename T>
__device__ __forceinline__ void gm_branch_c(T (&R)[4], const T* __restrict__ C, const T (&pi)[4]) {
    const T gR = fma(pi[2], R[2], pi[0] * R[0]);
    const T gY = fma(pi[3], R[3], pi[1] * R[1]);
    const T aT = C[0] * (gR + gY);
    const T xR = fma(C[1], gR, aT), xY = fma(C[2], gY, aT);
    R[0] = fma(C[3], R[0], xR);
    R[2] = fma(C[3], R[2], xR);
    R[1] = fma(C[4], R[1], xY);
    R[3] = fma(C[4], R[3], xY);
}
// column x of P(t) (the branch-transformed indicator of base x): P_{i x}
template <typename T>
__device__ __forceinline__ void gm_col_c(T (&v)[4], const T* __restrict__ C, int x, const T (&pi)[4]) {
    const int gx = x & 1;
#pragma unroll
    for (int i = 0; i < 4; ++i) {
        const int g = i & 1;
        T p = C[0] * pi[x];
        if (g == gx) p = fma(C[1 + g], pi[x], p);
        if (i == x) p += C[3 + g];
        v[i] = p;
    }
}

template <typename T, int D, int S, bool AMB>
__device__ __forceinline__ void gm_tt(T (&R)[D][4], uint32_t code, const T* __restrict__ P,
                                      const uint8_t* __restrict__ codes, int Lpad, int site, int& scale) {
    if constexpr (S < D) {
        int ta = (code >> 6) & 2047, tb = (code >> 17) & 2047;
        T va[4], vb[4];
        gm_tip<T, AMB>(va, P, __ldg(codes + (size_t)ta * Lpad + site));
        gm_tip<T, AMB>(vb, P + 16, __ldg(codes + (size_t)tb * Lpad + site));
#pragma unroll
        for (int i = 0; i < 4; ++i) R[S][i] = va[i] * vb[i];
        maybe_rescale(R[S], scale);
    }
}

template <typename T, int D, int S, bool AMB>
__device__ __forceinline__ void gm_ts(T (&R)[D][4], uint32_t code, const T* __restrict__ P,
                                      const uint8_t* __restrict__ codes, int Lpad, int site, int& scale) {
    if constexpr (S >= 1 && S <= D) {
        int ta = (code >> 6) & 2047;
        T va[4];
        gm_tip<T, AMB>(va, P, __ldg(codes + (size_t)ta * Lpad + site));
        gm_branch<T>(R[S - 1], P + 16);
#pragma unroll
        for (int i = 0; i < 4; ++i) R[S - 1][i] *= va[i];
        maybe_rescale(R[S - 1], scale);
    }
}

template <typename T, int D, int S>
__device__ __forceinline__ void gm_ss(T (&R)[D][4], const T* __restrict__ P, int& scale) {
    if constexpr (S >= 2 && S <= D) {
        gm_branch<T>(R[S - 2], P);
        gm_branch<T>(R[S - 1], P + 16);
#pragma unroll
        for (int i = 0; i < 4; ++i) R[S - 2][i] *= R[S - 1][i];
        maybe_rescale(R[S - 2], scale);
    }
}

#define MPCGS_GMCASE(S)                                                                       \
    case (OP_TT | ((S) << 2)): gm_tt<T, D, S, AMB>(R, code, P, codes, Lpad, site, scale); break; \
    case (OP_TS | ((S) << 2)): gm_ts<T, D, S, AMB>(R, code, P, codes, Lpad, site, scale); break; \
    case (OP_SS | ((S) << 2)): gm_ss<T, D, S>(R, P, scale); break;

// P matrices of every op's two children from the branch lengths in sched_e
// ({t_a, 0, t_b, 0} under the general model): one thread per (tree, op, child).
template <typename T>
__global__ void __launch_bounds__(128) k_pmat(const void* sched_e, const double* gm, T* sched_P, int nops,
                                              int ntrees) {
    __shared__ double sgm[36];
    if (threadIdx.x < 36) sgm[threadIdx.x] = gm[threadIdx.x];
    __syncthreads();
    const int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;  // (tree * nops + op) * 2 + child
    if (i >= (int64_t)ntrees * nops * 2) return;
    const T* e = reinterpret_cast<const T*>(sched_e) + (i >> 1) * 4;
    const double t = (double)e[(i & 1) ? 2 : 0];
    double P[16];
    pmat(sgm, t, P);
    T* out = sched_P + i * 16;
#pragma unroll
    for (int k = 0; k < 16; ++k) out[k] = (T)P[k];
}

#define MPCGS_OPCASE(S)                                                                     \
    case (OP_TT | ((S) << 2)): op_tt<T, D, S, AMB>(R, code, ed, codes, Lpad, site, pi, scale); break; \
    case (OP_TS | ((S) << 2)): op_ts<T, D, S, AMB>(R, code, ed, codes, Lpad, site, pi, scale); break; \
    case (OP_SS | ((S) << 2)): op_ss<T, D, S>(R, ed, pi, scale); break;

template <typename T, int D, bool W, bool GM, bool AMB>
__global__ void __launch_bounds__(PRUNE_THREADS) k_prune(PruneArgs a) {
    using E4 = typename Traits<T>::E4;
    extern __shared__ __align__(16) unsigned char smem_raw[];
    E4* s_e = reinterpret_cast<E4*>(smem_raw);
    uint32_t* s_op = reinterpret_cast<uint32_t*>(smem_raw + sizeof(E4) * a.nops);

    const int tree = blockIdx.y;
    const int tile = blockIdx.x;
    if (a.tree_need && a.tree_need[tree] <= a.need_cap) return;  // scored by the table pass
    const uint32_t* __restrict__ gop = a.sched_op + (size_t)tree * a.nops;
    const E4* __restrict__ ge = reinterpret_cast<const E4*>(a.sched_e) + (size_t)tree * a.nops;
    for (int i = threadIdx.x; i < a.nops; i += blockDim.x) {
        s_op[i] = gop[i];
        if constexpr (!GM) s_e[i] = ge[i];
    }
    __syncthreads();
    const T* __restrict__ gP = reinterpret_cast<const T*>(a.sched_P) + (size_t)tree * a.nops * 32;

    const T pi[4] = {(T)a.pi[0], (T)a.pi[1], (T)a.pi[2], (T)a.pi[3]};
    const uint8_t* __restrict__ codes = a.codes;
    const int Lpad = a.Lpad;
    int s_begin, s_end;
    tile_range(a, tile, s_begin, s_end);

    SiteAcc<W> acc;
    Exact128 ex;
    T R[D][4];
#pragma unroll
    for (int i = 0; i < D; ++i)
#pragma unroll
        for (int j = 0; j < 4; ++j) R[i][j] = T(0);

    // exact-sum units of FLAT_UNIT_SITES sites (tiles hold whole units, P22)
    for (int u0 = s_begin; u0 < s_end; u0 += FLAT_UNIT_SITES) {
        const int u1 = min(s_end, u0 + FLAT_UNIT_SITES);
        for (int site = u0 + threadIdx.x; site < u1; site += blockDim.x) {
            int scale = 0;
            for (int op = 0; op < a.nops; ++op) {
                const uint32_t code = s_op[op];
                if constexpr (GM) {
                    const T* __restrict__ P = gP + (size_t)op * 32;
                    switch (code & 63u) {
                        MPCGS_GMCASE(0) MPCGS_GMCASE(1) MPCGS_GMCASE(2) MPCGS_GMCASE(3) MPCGS_GMCASE(4)
                        MPCGS_GMCASE(5) MPCGS_GMCASE(6) MPCGS_GMCASE(7) MPCGS_GMCASE(8) MPCGS_GMCASE(9)
                        MPCGS_GMCASE(10) MPCGS_GMCASE(11)
                        default: break;
                    }
                } else {
                    const E4 ed = s_e[op];
                    switch (code & 63u) {
                        MPCGS_OPCASE(0) MPCGS_OPCASE(1) MPCGS_OPCASE(2) MPCGS_OPCASE(3) MPCGS_OPCASE(4)
                        MPCGS_OPCASE(5) MPCGS_OPCASE(6) MPCGS_OPCASE(7) MPCGS_OPCASE(8) MPCGS_OPCASE(9)
                        MPCGS_OPCASE(10) MPCGS_OPCASE(11)
                        default: break;
                    }
                }
            }
            // Eq. 21: L_s = sum_X pi_X L_root(X), root partial in R[0]
            T ls = pi[0] * R[0][0];
            ls = fma(pi[1], R[0][1], ls);
            ls = fma(pi[2], R[0][2], ls);
            ls = fma(pi[3], R[0][3], ls);
            acc.add((double)ls, scale, a.site_w, site);
        }
        // ln of this thread's product over the unit (0 if it had no site); -inf if a
        // site likelihood was 0 (S6)
        ex.add(acc.total());
        acc.reset();
    }
    __shared__ ExactScratch<PRUNE_THREADS> s_ex;
    exact_commit<PRUNE_THREADS>(ex, a.tree_acc + 4 * (size_t)tree, a.tile_cnt + tree, a.tiles,
                                a.out + (size_t)(a.out_first + tree) * a.out_stride, s_ex.w);
}

// ============================================================================
// Table kernel (the production path).  Tip codes are staged per site batch in
// shared memory (2-bit packed, cp.async double buffer); every tip child reads
// its 4-vector P_{.,x}(t) from a per-op 4x4 table and every cherry (two tip
// children) its product vector from a 16x4 table, both built in shared memory
// at CTA start; SI sites per thread are interleaved so that one dispatch and one
// read of the op serve SI register stacks.  The register stack holds DR levels;
// deeper levels (rare: need > DR) live in shared memory, so one compiled kernel
// scores every tree shape.
// ============================================================================
__device__ __forceinline__ void cp_async16(void* smem, const void* gmem) {
    unsigned sa = (unsigned)__cvta_generic_to_shared(smem);
    asm volatile("cp.async.cg.shared.global [%0], [%1], 16;\n" ::"r"(sa), "l"(gmem));
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;\n" ::); }
template <int N>
__device__ __forceinline__ void cp_async_wait() { asm volatile("cp.async.wait_group %0;\n" ::"n"(N)); }

// Shared-memory loads from 32-bit shared-window addresses: the op loop addresses
// its tables, code words and op records from one base computed before the loop
// (generic pointers made the compiler re-derive the shared window base per op).
__device__ __forceinline__ uint32_t smem_addr(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ uint32_t lds_u32(uint32_t a) {
    uint32_t v;
    asm volatile("ld.shared.u32 %0, [%1];\n" : "=r"(v) : "r"(a));
    return v;
}
__device__ __forceinline__ uint4 lds_u4(uint32_t a) {
    uint4 v;
    asm volatile("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];\n" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(a));
    return v;
}
__device__ __forceinline__ void lds2(double (&r)[2], uint32_t a) {
    asm volatile("ld.shared.v2.f64 {%0, %1}, [%2];\n" : "=d"(r[0]), "=d"(r[1]) : "r"(a));
}
__device__ __forceinline__ void lds2(float (&r)[2], uint32_t a) {
    asm volatile("ld.shared.v2.f32 {%0, %1}, [%2];\n" : "=f"(r[0]), "=f"(r[1]) : "r"(a));
}
__device__ __forceinline__ double lds1(uint32_t a, double) {
    double v;
    asm volatile("ld.shared.f64 %0, [%1];\n" : "=d"(v) : "r"(a));
    return v;
}
__device__ __forceinline__ float lds1(uint32_t a, float) {
    float v;
    asm volatile("ld.shared.f32 %0, [%1];\n" : "=f"(v) : "r"(a));
    return v;
}
__device__ __forceinline__ void sts1(uint32_t a, double v) { asm volatile("st.shared.f64 [%0], %1;\n" ::"r"(a), "d"(v)); }
__device__ __forceinline__ void sts1(uint32_t a, float v) { asm volatile("st.shared.f32 [%0], %1;\n" ::"r"(a), "f"(v)); }
__device__ __forceinline__ void lds4(double (&r)[4], uint32_t a) {
    asm volatile("ld.shared.v2.f64 {%0, %1}, [%2];\n" : "=d"(r[0]), "=d"(r[1]) : "r"(a));
    asm volatile("ld.shared.v2.f64 {%0, %1}, [%2+16];\n" : "=d"(r[2]), "=d"(r[3]) : "r"(a));
}
__device__ __forceinline__ void lds4(float (&r)[4], uint32_t a) {
    asm volatile("ld.shared.v4.f32 {%0, %1, %2, %3}, [%4];\n" : "=f"(r[0]), "=f"(r[1]), "=f"(r[2]), "=f"(r[3]) : "r"(a));
}

// FP64 tables in split-half layout: a table of E entries stores the first halves
// {v0, v1} of its entries (16 B each), then the second halves {v2, v3}.  A warp's
// 16-byte loads of data-dependent entries then spread over all 8 bank groups of a
// 128-byte row (contiguous 32-byte entries put every first half in an even group:
// about 1.4x the shared-memory wavefronts on random 16- and 64-entry gathers).
#ifndef MPCGS_SPLITTAB
#define MPCGS_SPLITTAB 1
#endif
template <typename T>
__host__ __device__ constexpr bool split_tab() { return MPCGS_SPLITTAB && sizeof(T) == 8; }
template <typename T>
__device__ __forceinline__ void tab_st(T* tab, int E, int i, const T (&v)[4]) {
    if constexpr (split_tab<T>()) {
        reinterpret_cast<double2*>(tab)[i] = make_double2(v[0], v[1]);
        reinterpret_cast<double2*>(tab)[E + i] = make_double2(v[2], v[3]);
    } else {
        st4<T>(tab + 4 * i, v);
    }
}
// entry of a table at byte address base: eo = the entry's index x 16 (split) or x 4 sizeof(T)
__device__ __forceinline__ void tab_ld(double (&r)[4], uint32_t a, uint32_t E) {
    if constexpr (split_tab<double>()) {
        asm volatile("ld.shared.v2.f64 {%0, %1}, [%2];\n" : "=d"(r[0]), "=d"(r[1]) : "r"(a));
        asm volatile("ld.shared.v2.f64 {%0, %1}, [%2];\n" : "=d"(r[2]), "=d"(r[3]) : "r"(a + 16u * E));
    } else {
        lds4(r, a);
    }
}
__device__ __forceinline__ void tab_ld(float (&r)[4], uint32_t a, uint32_t) { lds4(r, a); }

template <typename T, int SI>
__device__ __forceinline__ void rescale_sites(T (&v)[SI][4], int (&scale)[SI]) {
    bool any = false;
#pragma unroll
    for (int q = 0; q < SI; ++q) any |= small4(v[q]);
    if (__any_sync(0xffffffffu, any)) {
#pragma unroll
        for (int q = 0; q < SI; ++q) {
            const int k = rescale_k(v[q]);
            const T f = pow2(k, T(0));
            v[q][0] *= f; v[q][1] *= f; v[q][2] *= f; v[q][3] *= f;
            scale[q] += k;
        }
    }
}

// Register stack per site.  MPCGS_WINDOW (default): the registers hold the top
// DR levels (level l in register slot l mod DR, a compile-time index in every
// (sp, type) case); a push above DR spills the level leaving the window to shared
// memory and a merge that drops the window below its DR levels fills one back --
// one vector moved per crossing, not per op.  Otherwise levels >= DR live in shared
// memory for good.  Shared-memory levels are laid out [level][site k][state X][thread]
// (conflict-free).
#ifndef MPCGS_WINDOW
#define MPCGS_WINDOW 1
#endif

template <typename T, int DR, int SI>
struct Stack {
    T r[SI][DR][4];
    uint32_t sm;  // this thread's column of the spill area (shared-window address)
    __device__ __forceinline__ uint32_t sma(int level, int k, int x) const {
        return sm + (uint32_t)(((level * SI + k) * 4 + x) * PRUNE_THREADS) * (uint32_t)sizeof(T);
    }
    template <int S>
    __device__ __forceinline__ void get(int k, T (&v)[4]) const {
        if constexpr (MPCGS_WINDOW || S < DR) {
            constexpr int R = S % DR;
            v[0] = r[k][R][0]; v[1] = r[k][R][1]; v[2] = r[k][R][2]; v[3] = r[k][R][3];
        } else {
#pragma unroll
            for (int x = 0; x < 4; ++x) v[x] = lds1(sma(S - DR, k, x), T(0));
        }
    }
    template <int S>
    __device__ __forceinline__ void put(int k, const T (&v)[4]) {
        if constexpr (MPCGS_WINDOW || S < DR) {
            constexpr int R = S % DR;
            r[k][R][0] = v[0]; r[k][R][1] = v[1]; r[k][R][2] = v[2]; r[k][R][3] = v[3];
        } else {
#pragma unroll
            for (int x = 0; x < 4; ++x) sts1(sma(S - DR, k, x), v[x]);
        }
    }
    // before a push to level S: level S - DR leaves the window (slot S mod DR)
    template <int S>
    __device__ __forceinline__ void spill_for_push(int k) {
        if constexpr (MPCGS_WINDOW && S >= DR) {
#pragma unroll
            for (int x = 0; x < 4; ++x) sts1(sma(S - DR, k, x), r[k][S % DR][x]);
        }
    }
    // after a merge at stack depth S (levels S-2, S-1 -> S-2): level S-1-DR re-enters
    template <int S>
    __device__ __forceinline__ void fill_after_pop(int k) {
        if constexpr (MPCGS_WINDOW && S - 1 - DR >= 0) {
#pragma unroll
            for (int x = 0; x < 4; ++x) r[k][(S - 1) % DR][x] = lds1(sma(S - 1 - DR, k, x), T(0));
        }
    }
};

// Tip codes of the current site batch in shared memory, 2-bit packed, 16 sites
// per 32-bit word in the "thread-interleaved" order the host packs (codes2_pack):
// the word covering threads q = 0..16/SI-1 (SI sites each) holds site k of
// thread q at bit (32/SI) k + 2 q.  One shift and one mask leave a thread's SI
// codes as bytes (SI = 4: bytes 0..3; SI = 2: bytes 0 and 2), so the entry index
// of a cherry (4 a + b) or a fused triplet (16 a + 4 b + c) is formed for all SI
// sites at once with byte-lane arithmetic (no carries: every lane stays < 64).
// BITS = 4 (ambiguity codes): 4-bit base-set masks, 8 sites per
// word, site k of thread q at bit (32/SI) k + 4 q; the lanes are then 0..15.
template <int SI, int BITS = 2>
struct Codes {
    uint32_t sbase;             // this batch's buffer (shared-window address)
    int wofs;                   // word index of this thread's sites
    uint32_t qs;                // BITS q: this thread's bit offset in its word
    static constexpr int BATCH = PRUNE_THREADS * SI;
    static constexpr int SPW = 32 / BITS;          // sites per word
    static constexpr int WB = BATCH / SPW;         // words per tip row of a batch
    static constexpr uint32_t LM = (1u << BITS) - 1u;
    static constexpr uint32_t MASK = SI == 4 ? LM * 0x01010101u : LM * 0x00010001u;
    __device__ __forceinline__ void init(int tid) {
        wofs = (tid * SI) / SPW;
        qs = (uint32_t)BITS * (uint32_t)(tid % (SPW / SI));
    }
    __device__ __forceinline__ uint32_t word(int tip) const {
        return lds_u32(sbase + (uint32_t)(tip * WB + wofs) * 4u);
    }
    // this thread's SI codes of a word, one per byte lane
    __device__ __forceinline__ uint32_t lanes(uint32_t w) const { return (w >> qs) & MASK; }
    // byte offset of site k's entry in a table of EB-byte entries indexed by the lanes value
    template <int EB>
    __device__ __forceinline__ uint32_t off(uint32_t ln, int k) const {
        return __byte_perm(ln, 0u, 0x4440u + (uint32_t)(k * (4 / SI))) * (uint32_t)EB;
    }
    static constexpr size_t buf_bytes(int n) { return (size_t)n * WB * 4; }
};

constexpr uint32_t TAB_CHECK = 0x80000000u;  // toff flag: the cherry table can hold small vectors

// Sparse underflow checks (S5).  Every component of a branch-transformed child
// vector is >= d(child) * max(child), d = em * pi_min under F81 (Eq. 20: P_XY >=
// em pi_Y) or min_XY P_XY(t) under a general model, and a tip is a one-hot
// vector (max 1).  A node's vector is the product of its two transformed
// children, so log2 of its smallest component is bounded below by the sum of its
// children's bounds and ilogb(d_a) + ilogb(d_b).  mark_checks walks the schedule
// once per CTA with these integer bounds and sets OP_CHECK only on the ops whose
// result could otherwise come within reach of underflow; the check itself is
// unchanged (rescale by an exact power of two when max < 2^-TS), so the result
// is bit-identical to checking every node.
#ifndef MPCGS_SPARSE
#define MPCGS_SPARSE 1
#endif
#ifndef MPCGS_NO_TRIPLETS
#define MPCGS_NO_TRIPLETS 0
#endif
constexpr uint32_t OP_CHECK = 1u << 28;  // op code flag (bits 28-31 are free): check this op's result
// op code bits 29-30 of a TS-type op: 0 = tip table, 1 = fused cherry + SS, 2 = fused triplet + SS
constexpr int OP_FUSED_SHIFT = 29;
#ifndef MPCGS_FUSE_SS
#define MPCGS_FUSE_SS 1
#endif
// Fused triplet (table kernel only): a cherry (TT, tips a and b) immediately
// followed by the TS op that joins it to tip c -- one 64x4 table of the result
// over (x_a, x_b, x_c), built per CTA.  Type 3 is unused by the schedule encoding.
constexpr uint32_t OP_TTT = 3u;
constexpr int TRIP_EXTRA = 256 - 64 - 16;
// Code rows in consumption order (table kernel): the staged tip codes of a batch are
// laid out in the order the ops read the tips (each tip is read by exactly one op, in
// schedule order), so op i's words sit at rows k_i, k_i + 1, k_i + 2 with k_i a running
// count -- the code-word loads no longer wait for the op record.  `tc` carries k_i.
// Measured (interleaved A/B, profiles/r02_slot_rows_ab.txt): +3.7 % for the FP64 general
// model on 2-bit codes at need cap 4 (n <= 64; c5 F84 8.26 -> 7.95 ms); a loss for F81
// (FP64 -2.7 %, FP32 -5.6 %), FP32 F84 (-4.5 %), n = 128 / 256 HKY85 (-1.6 / -4 %) and
// 4-bit codes (-2.4 %) -- so that case only.
#ifndef MPCGS_SLOT_CODES
#define MPCGS_SLOT_CODES 1  // 0: off (tuning builds)
#endif
template <typename T, bool GM, int DMX, typename CD>
__host__ __device__ constexpr bool slot_rows() {
    return MPCGS_SLOT_CODES && GM && sizeof(T) == 8 && DMX == 4 && CD::SPW == 16;
}
#define MPCGS_ROW_B(code, tc) (slot_rows<T, GM, DMX, CD>() ? (int)(tc) + 1 : (int)(((code) >> 17) & 2047u))
#define MPCGS_ROW_C(tc) (slot_rows<T, GM, DMX, CD>() ? (int)(tc) + 2 : (int)(tc))
// tips an op reads (slot advance): TT 2, TS 1 / 2 / 3 (tip / fused cherry / fused triplet),
// SS 0, TTT 3; index = type | kind << 2 (two bits per entry)
__device__ __forceinline__ uint32_t op_tips(uint32_t x) {
    const uint32_t idx = (x & 3u) | (((x >> 29) & 3u) << 2);
    return (0x00CECAC6u >> (2u * idx)) & 3u;
}  // table values a fused triplet adds (64x4 vs 16x4 + 4x4)
constexpr int BOUND_NEG_INF = -100000;   // ilogb of 0 (or of a subnormal): no bound
// FP64 only: FP32's range leaves no room between checks (every op would be flagged)
template <typename T>
__host__ __device__ constexpr bool sparse_checks() { return MPCGS_SPARSE && sizeof(T) == 8; }

// unit-diagonal F81 branches in the table kernel (FP64; see prune_tab_body)
#ifndef MPCGS_UNITBR
#define MPCGS_UNITBR 1
#endif
#ifndef MPCGS_UNITBR32
#define MPCGS_UNITBR32 0  // FP32: measured -8 % at c5 (the second loop instance costs the issue-bound
                          // FP32 kernel more than the FMUL it saves; profiles/r02_kernel_iterations.md)
#endif
template <typename T, bool GM>
__host__ __device__ constexpr bool unit_branch() {
    return MPCGS_UNITBR && !GM && (sizeof(T) == 8 || MPCGS_UNITBR32);
}
// the unit form's growth budget in bits: a standard-form vector is < 2^(n-1) after
// power-of-two rescales, and the unit form multiplies it by at most 2^(-C / ln 2)
template <typename T>
__host__ __device__ constexpr int unit_budget_bits() { return sizeof(T) == 8 ? 900 : 120; }

template <typename T>
struct Bounds;
template <>
struct Bounds<double> {
    static constexpr int FLOOR = -1000;  // keep every component >= 2^-1000 (normal, 22 bits of margin)
    __device__ static int ilogb(double x) {
        const int ex = (__double2hiint(x) >> 20) & 2047;
        return (x > 0.0 && ex > 0) ? ex - 1023 : BOUND_NEG_INF;
    }
};
template <>
struct Bounds<float> {
    static constexpr int FLOOR = -120;
    __device__ static int ilogb(float x) {
        const int ex = (__float_as_int(x) >> 23) & 255;
        return (x > 0.0f && ex > 0) ? ex - 127 : BOUND_NEG_INF;
    }
};

// One warp: s_d[2 op + c] = lower bound of log2 d of child c of original op
// `op`; lpmin = ilogb(min pi) (the root's Eq. 21 dot product).  Walks the
// compacted op list s_opc (a fused triplet, type OP_TTT, covers original ops o
// and o+1) and sets s_chk[i] for the ops to check (merged into OP_CHECK later).
// compacted op record of the table kernel: {code, table byte offset, original op
// index, tip c of a fused triplet} and the op's up branch (one address, so the
// two loads of an op do not depend on each other)
template <typename T>
struct __align__(16) OpRec {
    uint4 h;
    T up[2];  // the op's up branch: F81 {e, em}; general model {offset of P_up in s_P, 0}
};

template <typename T>
__device__ void mark_checks(const OpRec<T>* s_opc, const int* s_d, unsigned char* s_chk, int nops_c, int lpmin,
                            int lane) {
    // one warp: the per-op data are loaded in parallel, lane l keeps the bound of
    // stack level l in a register, and the walk itself broadcasts op by op
    constexpr int TSX = Traits<T>::TS, FLOOR = Bounds<T>::FLOOR;
    auto dsum = [&](const uint4& o) {
        const int i = (int)o.z;
        int d = s_d[2 * i] + s_d[2 * i + 1];
        if ((o.x & 3u) == OP_TTT) d += s_d[2 * i + 2] + s_d[2 * i + 3];
        return d;
    };
    int dmax = 0;
    for (int i = lane; i < nops_c; i += 32) dmax = max(dmax, -dsum(s_opc[i].h));
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) dmax = max(dmax, __shfl_xor_sync(0xffffffffu, dmax, o));
    // stack entries stay >= limit, so an op's product is >= 2 limit - dmax >= FLOOR
    const int x = FLOOR + dmax;
    const int limit = x >= 0 ? (x + 1) / 2 : -((-x) / 2);
    const bool all = limit > -TSX;  // no room between checks (e.g. a zero-length branch): check every op
    int bnd = 0;                    // bound of stack level `lane`
    for (int base = 0; base < nops_c; base += 32) {
        const int i = base + lane;
        int ty = 0, sp = 0, ds = 0;
        if (i < nops_c) {
            const uint4 o = s_opc[i].h;
            ty = (int)(o.x & 3u);
            sp = (int)((o.x >> 2) & 15u);
            ds = dsum(o);
        }
        const int cnt = min(32, nops_c - base);
        bool mine = false;
        for (int q = 0; q < cnt; ++q) {
            const int qty = __shfl_sync(0xffffffffu, ty, q), qsp = __shfl_sync(0xffffffffu, sp, q);
            int b = __shfl_sync(0xffffffffu, ds, q);
            const int b1 = __shfl_sync(0xffffffffu, bnd, max(qsp - 1, 0));
            const int b2 = __shfl_sync(0xffffffffu, bnd, max(qsp - 2, 0));
            int slot;
            if (qty == (int)OP_TT || qty == (int)OP_TTT) {
                slot = qsp;
            } else if (qty == (int)OP_TS) {
                slot = qsp - 1;
                b += b1;
            } else {
                slot = qsp - 2;
                b += b2 + b1;
            }
            const bool chk = all || b < limit || (base + q == nops_c - 1 && b + lpmin < FLOOR);
            if (chk) b = -TSX;  // after the check: max >= 2^-TS
            if (lane == slot) bnd = b;
            if (lane == q) mine = chk;
        }
        if (i < nops_c) s_chk[i] = mine;
    }
}


// Every op pushes its node's vector already transformed by the node's own
// parent branch ("up" branch: branch(v)_X = sum_Y P_XY(t_up) v_Y, Eq. 19-20),
// so each edge of the tree is applied exactly once, by the op below it.  A
// cherry or fused-triplet table therefore stores branch_up(entry) -- its up
// branch costs nothing per site -- unless the table holds a vector small
// enough to need a rescale (TAB_CHECK, rare): then the raw entry is loaded,
// checked and transformed per site.  The up branch of the root op is the
// identity (e = 1, em = 0 / P = I), which leaves the root vector unchanged.
// U (unit-diagonal F81 branches, see unit_branch below): the record holds {1, r} with
// r = em / e, and the branch is v + r (pi . v) -- the e multiply is dropped.
template <typename T, bool GM, bool U = false>
struct UpBr {
    std::conditional_t<GM, const T*, T> e;
    T em;
    __device__ __forceinline__ UpBr(const T (&up)[2], const T* s_P) {
        if constexpr (GM) {
            e = s_P + (int)up[0];
        } else {
            e = up[0];
            em = up[1];
        }
    }
    __device__ __forceinline__ void apply(T (&v)[4], const T (&pi)[4]) const {
        if constexpr (GM) gm_branch_c<T>(v, e, pi);  // e -> the structured branch record
        else if constexpr (U) branch_unit<T>(v, em, pi);
        else branch<T>(v, e, em, pi);
    }
};

template <typename T, int DR, int SI, bool PT, int S, int DMX, bool GM, typename CD, typename UB>
__device__ __forceinline__ void tab_tt(Stack<T, DR, SI>& st, uint32_t code, uint32_t toff, uint32_t tc, uint32_t wa,
                                       const UB& ub, uint32_t s_tab, const CD& c,
                                       const T (&pi)[4], int (&scale)[SI]) {
    if constexpr (S < DMX) {
        constexpr int EB = split_tab<T>() ? 16 : 4 * sizeof(T);  // entry stride (split-half tables: 16)
        const uint32_t wb = c.word(MPCGS_ROW_B(code, tc));
        const uint32_t base = s_tab + (toff & ~TAB_CHECK);
        T v[SI][4];
        if constexpr (PT) {  // 16x4 table of the cherry, entry 4 x_a + x_b: branch_up(tip_a (.) tip_b)
            const uint32_t ix = (c.lanes(wa) << 2) + c.lanes(wb);
#pragma unroll
            for (int k = 0; k < SI; ++k) tab_ld(v[k], base + c.template off<EB>(ix, k), 16u);
            if (toff & TAB_CHECK) {  // raw table: check, then the up branch per site
                rescale_sites<T, SI>(v, scale);
#pragma unroll
                for (int k = 0; k < SI; ++k) ub.apply(v[k], pi);
            }
        } else {             // two 4x4 tip tables, multiplied here
            const uint32_t la = c.lanes(wa), lb = c.lanes(wb);
#pragma unroll
            for (int k = 0; k < SI; ++k) {
                T w[4];
                tab_ld(v[k], base + c.template off<EB>(la, k), CD::LM + 1u);
                tab_ld(w, base + 4u * (CD::LM + 1u) * (uint32_t)sizeof(T) + c.template off<EB>(lb, k), CD::LM + 1u);  // table b after a
#pragma unroll
                for (int i = 0; i < 4; ++i) v[k][i] *= w[i];
            }
            if (!sparse_checks<T>() || (code & OP_CHECK)) rescale_sites<T, SI>(v, scale);
#pragma unroll
            for (int k = 0; k < SI; ++k) ub.apply(v[k], pi);
        }
#pragma unroll
        for (int k = 0; k < SI; ++k) {
            st.template spill_for_push<S>(k);
            st.template put<S>(k, v[k]);
        }
    }
}

// fused triplet: one lookup in the 64x4 table of branch_up(tip(c) (.) branch(tip(a) (.) tip(b)))
template <typename T, int DR, int SI, bool PT, int S, int DMX, bool GM, typename CD, typename UB>
__device__ __forceinline__ void tab_ttt(Stack<T, DR, SI>& st, uint32_t code, uint32_t toff, uint32_t tc,
                                        uint32_t wa, const UB& ub, uint32_t s_tab, const CD& c,
                                        const T (&pi)[4], int (&scale)[SI]) {
    if constexpr (PT && S < DMX) {
        constexpr int EB = split_tab<T>() ? 16 : 4 * sizeof(T);
        const uint32_t wb = c.word(MPCGS_ROW_B(code, tc));
        const uint32_t wc = c.word(MPCGS_ROW_C(tc));
        const uint32_t base = s_tab + (toff & ~TAB_CHECK);
        T v[SI][4];
        const uint32_t ix = (c.lanes(wa) << 4) + (c.lanes(wb) << 2) + c.lanes(wc);  // entry 16 x_a + 4 x_b + x_c
#pragma unroll
        for (int k = 0; k < SI; ++k) tab_ld(v[k], base + c.template off<EB>(ix, k), 64u);
        if (toff & TAB_CHECK) {
            rescale_sites<T, SI>(v, scale);
#pragma unroll
            for (int k = 0; k < SI; ++k) ub.apply(v[k], pi);
        }
#pragma unroll
        for (int k = 0; k < SI; ++k) {
            st.template spill_for_push<S>(k);
            st.template put<S>(k, v[k]);
        }
    }
}

// tip a joined to the stack top (already carrying its branch): v = top (.) tip_a(x_a).
// Fused (OP_FUSED kind 1 / 2): a cherry / triplet table op and the SS that merges
// its result into the stack top, v = top (.) table(x_a, x_b[, x_c]) -- the table
// already carries the cherry's branch into the SS, the op record the SS's up branch.
template <typename T, int DR, int SI, int S, int DMX, bool GM, typename CD, typename UB>
__device__ __forceinline__ void tab_ts(Stack<T, DR, SI>& st, uint32_t code, uint32_t toff, uint32_t tc,
                                       uint32_t wa, const UB& ub, uint32_t s_tab, const CD& c,
                                       const T (&pi)[4], int (&scale)[SI]) {
    if constexpr (S >= 1 && S <= DMX) {
        constexpr int EB = split_tab<T>() ? 16 : 4 * sizeof(T);
        const uint32_t base = s_tab + (toff & ~TAB_CHECK);
        uint32_t la = c.lanes(wa);
        const uint32_t kind = (code >> OP_FUSED_SHIFT) & 3u;
        const uint32_t E = (CD::LM + 1u) << (2u * kind);  // tip 4 (16 base sets), cherry 16, triplet 64
        if (kind != 0u) {
            la = (la << 2) + c.lanes(c.word(MPCGS_ROW_B(code, tc)));
            if (kind == 2u) la = (la << 2) + c.lanes(c.word(MPCGS_ROW_C(tc)));
        }
        T v[SI][4];
#pragma unroll
        for (int k = 0; k < SI; ++k) {
            T tip[4];
            tab_ld(tip, base + c.template off<EB>(la, k), E);
            st.template get<S - 1>(k, v[k]);
#pragma unroll
            for (int i = 0; i < 4; ++i) v[k][i] *= tip[i];
        }
        if (!sparse_checks<T>() || (code & OP_CHECK)) rescale_sites<T, SI>(v, scale);
#pragma unroll
        for (int k = 0; k < SI; ++k) {
            ub.apply(v[k], pi);
            st.template put<S - 1>(k, v[k]);
        }
    }
}

// two stack entries (each already carrying its branch): v = second (.) top
template <typename T, int DR, int SI, int S, int DMX, bool GM, typename UB>
__device__ __forceinline__ void tab_ss(Stack<T, DR, SI>& st, uint32_t code, const UB& ub,
                                       const T (&pi)[4], int (&scale)[SI]) {
    if constexpr (S >= 2 && S <= DMX) {
        T v[SI][4];
#pragma unroll
        for (int k = 0; k < SI; ++k) {
            T w[4];
            st.template get<S - 2>(k, v[k]);
            st.template get<S - 1>(k, w);
#pragma unroll
            for (int i = 0; i < 4; ++i) v[k][i] *= w[i];
        }
        if (!sparse_checks<T>() || (code & OP_CHECK)) rescale_sites<T, SI>(v, scale);
#pragma unroll
        for (int k = 0; k < SI; ++k) {
            ub.apply(v[k], pi);
            st.template put<S - 2>(k, v[k]);
            st.template fill_after_pop<S>(k);
        }
    }
}

#define MPCGS_TABCASE(S)                                                                          \
    case 4 * (S) + 0: tab_tt<T, DR, SI, PT, S, DMX, GM, CD>(st, code, toff, tc, wa, ub, s_tab, cc, pi, scale); break;       \
    case 4 * (S) + 1: tab_ts<T, DR, SI, S, DMX, GM, CD>(st, code, toff, tc, wa, ub, s_tab, cc, pi, scale); break; \
    case 4 * (S) + 2: tab_ss<T, DR, SI, S, DMX, GM>(st, code, ub, pi, scale); break;                      \
    case 4 * (S) + 3: tab_ttt<T, DR, SI, PT, S, DMX, GM, CD>(st, code, toff, tc, wa, ub, s_tab, cc, pi, scale); break;
#define MPCGS_CASES_4 MPCGS_TABCASE(0) MPCGS_TABCASE(1) MPCGS_TABCASE(2) MPCGS_TABCASE(3) MPCGS_TABCASE(4)
#define MPCGS_CASES_6 MPCGS_CASES_4 MPCGS_TABCASE(5) MPCGS_TABCASE(6)
#define MPCGS_CASES_8 MPCGS_CASES_6 MPCGS_TABCASE(7) MPCGS_TABCASE(8)
#define MPCGS_CASES_10 MPCGS_CASES_8 MPCGS_TABCASE(9) MPCGS_TABCASE(10)

// one op for SI sites; the switch only has the (sp, type) labels a DMX-level tree can use
template <typename T, int DR, int SI, bool PT, int DMX, bool GM, typename CD, typename UB>
__device__ __forceinline__ void run_op(int di, Stack<T, DR, SI>& st, uint32_t code, uint32_t toff, uint32_t tc,
                                       uint32_t wa, const UB& ub, uint32_t s_tab, const CD& cc,
                                       const T (&pi)[4], int (&scale)[SI]) {
    if constexpr (DMX <= 4) {
        switch (di) { MPCGS_CASES_4 default: __builtin_unreachable(); }
    } else if constexpr (DMX <= 6) {
        switch (di) { MPCGS_CASES_6 default: __builtin_unreachable(); }
    } else if constexpr (DMX <= 8) {
        switch (di) { MPCGS_CASES_8 default: __builtin_unreachable(); }
    } else {
        switch (di) { MPCGS_CASES_10 default: __builtin_unreachable(); }
    }
}

__host__ __device__ constexpr size_t align16(size_t x) { return (x + 15) & ~(size_t)15; }

// Shared-memory layout of the table kernel for trees of n tips whose register need is
// at most `need` (spill levels above DR), with up to `trip_cap` fused triplets and
// `bufs` tip-code staging buffers.  F81: the per-op branch data s_e and the setup
// arrays s_d / s_tl are dead once the op loop starts, so they live in space the loop
// only needs later -- the second code buffer (double buffering: first filled by the
// prefetch of batch 1, after the setup) or the shared spill levels (single buffer).
// bufs = 1 is chosen where it buys a resident CTA per SM (n = 256: 2 -> 3).
#ifndef MPCGS_ALIAS
#define MPCGS_ALIAS 1
#endif
#ifndef MPCGS_SINGLEBUF
#define MPCGS_SINGLEBUF 1
#endif
#ifndef MPCGS_GM32_MAXCTA
#define MPCGS_GM32_MAXCTA 4
#endif
template <typename T, int DR, int SI, bool PT, bool GM = false, int BITS = 2>
struct TabLayout {
    size_t e, tab, opc, cod, bufb, spill, d, tl, pos, total;
    __host__ __device__ TabLayout(int nops, int need, int trip_cap, int bufs) {
        const int n = nops + 1;
        const size_t e_bytes = align16(GM ? 2 * GMC * sizeof(T) * nops + GMC * sizeof(T)
                                          : sizeof(typename Traits<T>::E4) * nops);
        const size_t d_bytes = align16(sizeof(int) * 2 * (size_t)nops), tl_bytes = align16(sizeof(int) * (size_t)nops);
        const size_t spill_bytes = sizeof(T) * (size_t)(need > DR ? need - DR : 0) * SI * 4 * PRUNE_THREADS;
        const size_t scratch = e_bytes + d_bytes + tl_bytes;
        bufb = align16(Codes<SI, BITS>::buf_bytes(n));
        const bool in_buf1 = MPCGS_ALIAS && !GM && bufs == 2 && scratch <= bufb;
        const bool in_spill = MPCGS_ALIAS && !GM && !in_buf1 && scratch <= spill_bytes;
        size_t o = 0;
        e = 0;
        if (!in_buf1 && !in_spill) o += e_bytes;
        tab = o;
        o += align16(sizeof(T) * ((PT ? 32 : (BITS == 4 ? 64 : 16)) * (size_t)n + (size_t)TRIP_EXTRA * (PT ? trip_cap : 0)));
        opc = o;
        o += align16(sizeof(OpRec<T>) * nops);
        cod = o;
        o += (size_t)bufs * bufb;
        spill = o;
        o += spill_bytes;
        if (in_buf1 || in_spill) {
            e = in_buf1 ? cod + bufb : spill;
            d = e + e_bytes;
            tl = d + d_bytes;
        } else {
            d = o;
            tl = d + d_bytes;
            o = tl + tl_bytes;
        }
        pos = o;  // tip -> code row (slot_rows only)
        if (GM && sizeof(T) == 8 && BITS == 2) o += align16(sizeof(int) * (size_t)(nops + 1));
        total = o + 64 * sizeof(int);
    }
};
template <typename T, int DR, int SI, bool PT, bool GM = false, int BITS = 2>
__host__ __device__ size_t tab_smem_bytes(int nops, int need, int trip_cap, int bufs = 2) {
    return TabLayout<T, DR, SI, PT, GM, BITS>(nops, need, trip_cap, bufs).total;
}

#ifdef MPCGS_MINB  // tuning builds only: min CTAs per SM (caps registers)
#define MPCGS_TAB_BOUNDS __launch_bounds__(PRUNE_THREADS, MPCGS_MINB)
#else
// FP64: hold the register budget at 3 CTAs per SM (<= 168 registers).  The general
// model (F84 / HKY85) would take 204 and fall to 2 CTAs (c5 F84 9.63 -> 8.27 ms per
// step); the F81 kernel uses the room for scheduling (159 -> 165, 6.29 -> 6.20 ms).
// FP32 is left free (minBlocks 0: a cap of 3 raised it from 96 to 118 registers, -0.6 %).
#define MPCGS_TAB_BOUNDS __launch_bounds__(PRUNE_THREADS, sizeof(T) == 8 ? 3 : 0)
#endif
#ifdef MPCGS_PRUNE_TS  // diagnosis: setup phase cycles of CTA (0, 0), printed once per launch
static __device__ long long g_pts[8];
#define PTS(i) do { if (threadIdx.x == 0 && blockIdx.x == 0 && blockIdx.y == 0) g_pts[i] = clock64(); } while (0)
#else
#define PTS(i) do { } while (0)
#endif

// One CTA scores genealogy `tree` over site tile `tile`; its schedule is gop / ge
// (global memory written by k_propose); smem_raw = the
// dynamic shared memory of tab_smem_bytes.
template <typename T, int DR, int SI, bool PT, int DMX, bool W, bool GM, int BITS, bool UK>
__device__ __forceinline__ void prune_tab_body(const PruneArgs& a, int tree, int tile, const uint32_t* gop,
                                               const typename Traits<T>::E4* ge, unsigned char* smem_raw) {
    using E4 = typename Traits<T>::E4;
    using CD = Codes<SI, BITS>;
    static_assert(BITS == 2 || !PT, "4-bit (ambiguity) codes use tip tables only");
    constexpr uint32_t TABE = PT ? 32u : (BITS == 4 ? 64u : 16u);  // table values per tip
    constexpr int BATCH = CD::BATCH;  // sites per batch
    constexpr size_t OPB = GM ? 2 * GMC * sizeof(T) : sizeof(E4);  // branch data bytes per op
    const int nops = a.nops, n = nops + 1;
    const int trip_cap = PT ? a.trip_cap : 0;
    const int bufs = a.code_bufs == 1 ? 1 : 2;
    const TabLayout<T, DR, SI, PT, GM, BITS> lay(nops, a.need_cap, trip_cap, bufs);
    E4* s_e = reinterpret_cast<E4*>(smem_raw + lay.e);  // F81: {e_a, em_a, e_b, em_b} per op
    T* s_P = reinterpret_cast<T*>(smem_raw + lay.e);    // general model: branch records {C_a, C_b} per op
    // general model: {C_a, C_b} of every op, then the identity record (the root's up branch)
    T* s_tab = reinterpret_cast<T*>(smem_raw + lay.tab);
    // compacted ops: {code, table byte offset, original op index, tip c of a fused triplet}
    OpRec<T>* s_opc = reinterpret_cast<OpRec<T>*>(smem_raw + lay.opc);
    unsigned char* s_cod = smem_raw + lay.cod;
    const size_t bufb = lay.bufb;
    T* s_spill = reinterpret_cast<T*>(smem_raw + lay.spill);
    int* s_d = reinterpret_cast<int*>(smem_raw + lay.d);
    int* s_tl = reinterpret_cast<int*>(smem_raw + lay.tl);  // original codes, then check flags
    // tip -> code row (slot_rows only: reserved for FP64 general-model 2-bit kernels; every
    // byte here costs the others triplet tables, FP32 c5 -3.8 % with it)
    int* s_pos = reinterpret_cast<int*>(smem_raw + lay.pos);
    __shared__ int s_nc;  // compacted op count

    const int tid = threadIdx.x;
    int s_begin, s_end;
    tile_range(a, tile, s_begin, s_end);
    const int nb = (s_end - s_begin + BATCH - 1) / BATCH;
    PTS(0);

    auto issue = [&](int b, int buf) {
        const int site0 = s_begin + b * BATCH;
        unsigned char* dst = s_cod + (size_t)buf * bufb;
        constexpr int WB = CD::WB, CH = WB / 4;  // 16-byte chunks per tip row
        const uint32_t* src = a.codes2 + site0 / CD::SPW;
        for (int c = tid; c < n * CH; c += PRUNE_THREADS) {
            const int tip = c / CH, q = c - tip * CH;
            const int row = slot_rows<T, GM, DMX, CD>() ? s_pos[tip] : tip;
            cp_async16(dst + ((size_t)row * WB + q * 4) * 4, src + (size_t)tip * a.W2 + q * 4);
        }
        cp_async_commit();
    };
    if (!slot_rows<T, GM, DMX, CD>() && nb > 0) issue(0, 0);  // (slot rows: after the scan below lays them out)

    // 1. schedule, branch data and the per-child bounds d (mark_checks, fusion guard)
    const T pi[4] = {(T)a.pi[0], (T)a.pi[1], (T)a.pi[2], (T)a.pi[3]};
    const T pimin = min(min(pi[0], pi[1]), min(pi[2], pi[3]));
    uint32_t* s_code = reinterpret_cast<uint32_t*>(s_tl);  // original codes (s_tl is filled after the scan)
    double lne = 0.0;  // unit branches: this thread's sum of ln e over its ops' two child branches
    for (int i = tid; i < nops; i += PRUNE_THREADS) {
        s_code[i] = gop[i];
        if constexpr (!GM) {  // d = em pi_min (Eq. 20)
            const E4 ed = ge[i];
            s_e[i] = ed;
            const int lp = Bounds<T>::ilogb(pimin);
            s_d[2 * i] = Bounds<T>::ilogb((T)ed.y) + lp;
            s_d[2 * i + 1] = Bounds<T>::ilogb((T)ed.w) + lp;
            if constexpr (UK && unit_branch<T, GM>())
                if (a.unit_form) lne += log((double)ed.x) + log((double)ed.z);
        }
    }
    // Unit-diagonal branches (F81, FP64): every branch b of the tree is applied divided
    // by its e_b, so a vector carries the factor 1 / prod e_b of the branches below it
    // and the root 1 / prod_b e_b, the same at every site: ln L_s = ln(pi . root_s) +
    // scale_s ln 2 + C with C = sum_b ln e_b = -u (tree length), added once per tree
    // (exact_commit).  Those factors only enlarge vectors (the S5 lower bounds stay
    // valid); the form is used while they cannot overflow: -C / ln 2 <= 900 - n bits (FP32: 120 - n)
    // (a vector of the standard form is < 2^(n-1) after power-of-two rescales), else
    // the tree keeps the standard branch.  C is reduced in a fixed order, so every CTA
    // of a tree (any tiling, any world size) adds the same double (P22).
    bool unit = false;
    double lnC = 0.0;
    if constexpr (UK && unit_branch<T, GM>()) if (a.unit_form) {
        __shared__ double s_lne[PRUNE_THREADS / 32];
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) lne += __shfl_down_sync(0xffffffffu, lne, o);
        if ((tid & 31) == 0) s_lne[tid >> 5] = lne;
        __syncthreads();
        lnC = s_lne[0];
#pragma unroll
        for (int w = 1; w < PRUNE_THREADS / 32; ++w) lnC += s_lne[w];
        unit = -lnC * 1.4426950408889634 <= (double)(unit_budget_bits<T>() - n);  // false for -inf / NaN
        if (unit) {
            for (int i = tid; i < nops; i += PRUNE_THREADS) {
                E4 ed = s_e[i];
                ed.y = ed.y / ed.x;  // {1, r = em / e} per side
                ed.w = ed.w / ed.z;
                ed.x = (T)1;
                ed.z = (T)1;
                s_e[i] = ed;
            }
        } else {
            lnC = 0.0;
        }
    }
    if constexpr (GM) {  // {C_a, C_b} of every op from its branch lengths {t_a, 0, t_b, 0}; d = min_XY P_XY(t)
        for (int i = tid; i < nops * 2; i += PRUNE_THREADS) {
            const E4 ed = ge[i >> 1];
            T* C = s_P + i * GMC;
            gm_coef<T>(a.gm + 36, (double)((i & 1) ? ed.z : ed.x), C);
            T pmin = T(1);
#pragma unroll
            for (int x = 0; x < 4; ++x) {
                T col[4];
                gm_col_c<T>(col, C, x, pi);
                pmin = min(pmin, min(min(col[0], col[1]), min(col[2], col[3])));
            }
            s_d[i] = Bounds<T>::ilogb(pmin);
        }
        if (tid < GMC) s_P[nops * 2 * GMC + tid] = (tid == 3 || tid == 4) ? T(1) : T(0);  // identity: a = b = 0, c = 1
    }
    __syncthreads();
    PTS(2);
    // 2. warp 0: fuse the first trip_cap (TT, TS) pairs, compact the op list and
    //    lay out the tables (exclusive scans over the original ops)
    if (tid < 32) {
        uint32_t c_keep = 0, c_size = 0, c_cand = 0, prev_start = 0, c_rows = 0;
        for (int base = 0; base < nops; base += 32) {
            const int i = base + tid;
            uint32_t code = 0, ty = 2, tyn = 2;
            if (i < nops) {
                code = s_code[i];
                ty = code & 3u;
                if (i + 1 < nops) tyn = s_code[i + 1] & 3u;
            }
            // candidate: a cherry whose parent joins it to a tip, with table values safely normal
            const bool cand = PT && i < nops && ty == OP_TT && tyn == OP_TS &&
                              s_d[2 * i] + s_d[2 * i + 1] + s_d[2 * i + 2] + s_d[2 * i + 3] >= Bounds<T>::FLOOR / 2;
            const unsigned mc = __ballot_sync(0xffffffffu, cand);
            const uint32_t rank = c_cand + __popc(mc & ((1u << tid) - 1u));
            const bool start = cand && rank < (uint32_t)trip_cap;
            const unsigned ms = __ballot_sync(0xffffffffu, start);
            const bool prev = tid == 0 ? prev_start != 0u : ((ms >> (tid - 1)) & 1u) != 0u;
            const bool keep = i < nops && !(ty == OP_TS && prev);
            uint32_t sz = 0;
            if (keep) sz = start ? 256u : (ty == OP_TT ? 2u * TABE : (ty == OP_TS ? (BITS == 4 ? 64u : 16u) : 0u));
            const unsigned mk = __ballot_sync(0xffffffffu, keep);
            const uint32_t j = c_keep + __popc(mk & ((1u << tid) - 1u));
            uint32_t x = sz;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
                if (tid >= o) x += y;
            }
            const uint32_t tc = (i + 1 < nops) ? ((s_code[i + 1] >> 6) & 2047u) : 0u;
            if (slot_rows<T, GM, DMX, CD>()) {  // code rows in consumption order: TT reads (a, b), TS reads a
                const uint32_t nt = i < nops ? (ty == OP_TT ? 2u : (ty == OP_TS ? 1u : 0u)) : 0u;
                uint32_t y = nt;
#pragma unroll
                for (int o = 1; o < 32; o <<= 1) {
                    const uint32_t z = __shfl_up_sync(0xffffffffu, y, o);
                    if (tid >= o) y += z;
                }
                const uint32_t row = c_rows + y - nt;
                if (nt >= 1u) s_pos[(code >> 6) & 2047u] = (int)row;
                if (nt == 2u) s_pos[(code >> 17) & 2047u] = (int)row + 1;
                c_rows += __shfl_sync(0xffffffffu, y, 31);
            }
            __syncwarp();
            if (keep) {
                const uint32_t cx = start ? ((code & ~3u) | OP_TTT) : code;
                s_opc[j].h = make_uint4(cx, (c_size + x - sz) * (uint32_t)sizeof(T), (uint32_t)i, start ? tc : 0u);
            }
            c_size += __shfl_sync(0xffffffffu, x, 31);
            c_keep += __popc(mk);
            c_cand += __popc(mc);
            prev_start = (ms >> 31) & 1u;
        }
        if (tid == 0) s_nc = (int)c_keep;
    }
    __syncthreads();
    PTS(3);
    if (slot_rows<T, GM, DMX, CD>() && nb > 0) issue(0, 0);
    const int nops_c = s_nc;
    // 3. sparse checks (FP64): warp 1 walks the bounds while the others build the tables
    unsigned char* s_chk = reinterpret_cast<unsigned char*>(s_tl);  // s_code is dead after the scan
    if constexpr (sparse_checks<T>()) {
        if (tid >= 32 && tid < 64) mark_checks<T>(s_opc, s_d, s_chk, nops_c, Bounds<T>::ilogb(pimin), tid - 32);
    }
    //    up branch of every op: the child branch its consumer (the first later op
    //    that pops the level it pushes) applies to it -- side a of an SS for the
    //    second entry, side b for the top (SS) or the subtree (TS); none (the
    //    identity) for the root.  Stored in the op record in place of the
    //    children's branch data, which the per-site path no longer needs.
    // (warps other than the bound-walking warp 1 share the ops)
    constexpr int NSCAN = sparse_checks<T>() ? PRUNE_THREADS - 32 : PRUNE_THREADS;
    const int tscan = (sparse_checks<T>() && tid >= 64) ? tid - 32 : tid;
    for (int i = tscan; i < nops_c && !(sparse_checks<T>() && tid >= 32 && tid < 64); i += NSCAN) {
        const uint32_t xi = s_opc[i].h.x;
        const int ty = (int)(xi & 3u), sp = (int)((xi >> 2) & 15u);
        const int lvl = (ty == (int)OP_TS) ? sp - 1 : (ty == (int)OP_SS ? sp - 2 : sp);
        T up0 = GM ? (T)(nops * 2 * GMC) : T(1), up1 = T(0);
        for (int j = i + 1; j < nops_c; ++j) {
            const uint4 oj = s_opc[j].h;
            const int tj = (int)(oj.x & 3u), sj = (int)((oj.x >> 2) & 15u);
            const int side = (tj == (int)OP_TS && sj - 1 == lvl) ? 1
                             : (tj == (int)OP_SS && sj - 2 == lvl) ? 0
                             : (tj == (int)OP_SS && sj - 1 == lvl) ? 1 : -1;
            if (side < 0) continue;
            if constexpr (GM) {
                up0 = (T)(oj.z * 2u * GMC + (uint32_t)side * GMC);
            } else {
                const E4 e = s_e[oj.z];
                up0 = side ? (T)e.z : (T)e.x;
                up1 = side ? (T)e.w : (T)e.y;
            }
            break;
        }
        s_opc[i].up[0] = up0;
        s_opc[i].up[1] = up1;
    }
    __syncthreads();  // every op's up branch is in place
    PTS(4);
    //    tables, one row per work item: tip tables P_{.,x}(t) (Eq. 19-20 at an indicator
    //    tip), cherry rows tip_a(xa) (.) tip_b(xb), and fused-triplet rows tip_c(xc) (.)
    //    branch(tip_a(xa) (.) tip_b(xb)) for the four xc -- the TS op applied to the
    //    cherry's vector, as the per-site path computes it.
    // 4. cherry / triplet tables are stored with their op's up branch folded in, unless
    //    an entry is small enough to need a rescale (max < 2^-TS): that table stays raw
    //    and is checked and transformed per site (TAB_CHECK).  A half warp (16 lanes,
    //    rows r) covers one op, so the flag is one ballot; each entry is stored once.
    const int nrow = ((nops_c * 16 + 31) / 32) * 32;
    for (int idx = tid; idx < nrow; idx += PRUNE_THREADS) {
        const int op = idx >> 4, r = idx & 15;
        bool tabop = false, small = false;  // tabop: a cherry / triplet table to fold (PT)
        int ne = 1;
        T* tab = nullptr;
        T v[4][4];
        if (op < nops_c) {
            const uint4 ox = s_opc[op].h;
            const uint32_t ty = ox.x & 3u;
            tab = reinterpret_cast<T*>(reinterpret_cast<char*>(s_tab) + (ox.y & ~TAB_CHECK));
            T va[4], vb[4];
            if constexpr (GM) {  // tip vectors are columns of P (row X = parent state)
                const T* Ca = s_P + ox.z * 2 * GMC;
                if (ty == OP_TT && PT) {
                    gm_col_c<T>(va, Ca, r >> 2, pi);
                    gm_col_c<T>(vb, Ca + GMC, r & 3, pi);
#pragma unroll
                    for (int X = 0; X < 4; ++X) v[0][X] = va[X] * vb[X];
                    tabop = true;
                } else if (BITS == 4 && (ty == OP_TT || ty == OP_TS)) {  // 16-row base-set tables (S24)
                    auto setcol = [&](T (&w)[4], const T* C, int m) {
#pragma unroll
                        for (int X = 0; X < 4; ++X) w[X] = T(0);
#pragma unroll
                        for (int x = 0; x < 4; ++x)
                            if ((m >> x) & 1) {
                                T col[4];
                                gm_col_c<T>(col, C, x, pi);
#pragma unroll
                                for (int X = 0; X < 4; ++X) w[X] += col[X];
                            }
                    };
                    setcol(va, Ca, r);
                    tab_st<T>(tab, 16, r, va);
                    if (ty == OP_TT) {  // table b after table a
                        setcol(vb, Ca + GMC, r);
                        tab_st<T>(tab + 16 * 4, 16, r, vb);
                    }
                } else if (ty == OP_TT && r < 8) {
                    gm_col_c<T>(va, Ca + (r < 4 ? 0 : GMC), r & 3, pi);
                    tab_st<T>(tab + (r & 4) * 4, 4, r & 3, va);
                } else if (ty == OP_TS && r < 4) {
                    gm_col_c<T>(va, Ca, r, pi);
                    tab_st<T>(tab, 4, r, va);
                } else if (ty == OP_TTT) {  // op o: C_a, C_b; op o+1: C of tip c, C of the cherry's branch
                    const T* Cc = Ca + 2 * GMC;
                    gm_col_c<T>(va, Ca, r >> 2, pi);
                    gm_col_c<T>(vb, Ca + GMC, r & 3, pi);
#pragma unroll
                    for (int X = 0; X < 4; ++X) va[X] *= vb[X];
                    gm_branch_c<T>(va, Cc + GMC, pi);
#pragma unroll
                    for (int xc = 0; xc < 4; ++xc) {
                        gm_col_c<T>(vb, Cc, xc, pi);
#pragma unroll
                        for (int X = 0; X < 4; ++X) v[xc][X] = vb[X] * va[X];
                    }
                    tabop = true;
                    ne = 4;
                }
            } else {
                const E4 ed = s_e[ox.z];
                if (ty == OP_TT && PT) {
                    tipvec<T>(va, r >> 2, (T)ed.x, (T)ed.y, pi);
                    tipvec<T>(vb, r & 3, (T)ed.z, (T)ed.w, pi);
#pragma unroll
                    for (int X = 0; X < 4; ++X) v[0][X] = va[X] * vb[X];
                    tabop = true;
                } else if (BITS == 4 && (ty == OP_TT || ty == OP_TS)) {  // 16-row base-set tables (S24)
                    tip81<T, true>(va, r, (T)ed.x, (T)ed.y, pi);          // e [X in set] + em pi(set)
                    tab_st<T>(tab, 16, r, va);
                    if (ty == OP_TT) {
                        tip81<T, true>(vb, r, (T)ed.z, (T)ed.w, pi);
                        tab_st<T>(tab + 16 * 4, 16, r, vb);
                    }
                } else if (ty == OP_TT && r < 8) {  // two tip tables: a at [0, 16), b at [16, 32)
                    if (r < 4) tipvec<T>(va, r, (T)ed.x, (T)ed.y, pi);
                    else tipvec<T>(va, r - 4, (T)ed.z, (T)ed.w, pi);
                    tab_st<T>(tab + (r & 4) * 4, 4, r & 3, va);
                } else if (ty == OP_TS && r < 4) {
                    tipvec<T>(va, r, (T)ed.x, (T)ed.y, pi);
                    tab_st<T>(tab, 4, r, va);
                } else if (ty == OP_TTT) {
                    const E4 e1 = s_e[ox.z + 1];
                    tipvec<T>(va, r >> 2, (T)ed.x, (T)ed.y, pi);
                    tipvec<T>(vb, r & 3, (T)ed.z, (T)ed.w, pi);
#pragma unroll
                    for (int X = 0; X < 4; ++X) va[X] *= vb[X];
                    branch<T>(va, (T)e1.z, (T)e1.w, pi);
#pragma unroll
                    for (int xc = 0; xc < 4; ++xc) {
                        tipvec<T>(vb, xc, (T)e1.x, (T)e1.y, pi);
#pragma unroll
                        for (int X = 0; X < 4; ++X) v[xc][X] = vb[X] * va[X];
                    }
                    tabop = true;
                    ne = 4;
                }
            }
#pragma unroll
            for (int e = 0; e < 4; ++e)
                if (tabop && e < ne) small |= small4(v[e]);
        }
        const unsigned m = __ballot_sync(0xffffffffu, small);
        const bool raw = ((m >> (tid & 16)) & 0xffffu) != 0u;
        if (tabop) {
            if (raw) {
                if (r == 0) s_opc[op].h.y |= TAB_CHECK;
            } else {
                const UpBr<T, GM> ub(s_opc[op].up, s_P);
#pragma unroll
                for (int e = 0; e < 4; ++e)
                    if (e < ne) ub.apply(v[e], pi);
            }
#pragma unroll
            for (int e = 0; e < 4; ++e)
                if (e < ne) tab_st<T>(tab, ne == 4 ? 64 : 16, r * ne + e, v[e]);  // cherry 16, triplet 64 entries
        }
    }
    // the check flags are merged into the op codes after this pass (which reads the
    // codes): by the fusion warp below, or by this loop when there is no fusion
    if constexpr (sparse_checks<T>() && !(PT && MPCGS_FUSE_SS)) {  // ordered before the op loop by the batch barrier
        __syncthreads();
        for (int op = tid; op < nops_c; op += PRUNE_THREADS)
            if (s_chk[op]) s_opc[op].h.x |= OP_CHECK;
    }
    PTS(5);
    // 5. fuse each folded cherry / triplet op with an SS that immediately merges its
    //    result: one TS-type op at the table op's depth (top (.) table entry) with the
    //    SS's check flag and up branch -- one dispatch, push and pop fewer per pair.
    int nops_run = nops_c;
    if constexpr (PT && MPCGS_FUSE_SS) {
        __syncthreads();
        if (tid < 32) {  // warp 0: ballot compaction, in place (every write index <= its read index)
            uint32_t c_keep = 0;
            bool carry = false;
            for (int base = 0; base < nops_c; base += 32) {
                const int i = base + tid;
                OpRec<T> o;
                bool head = false;
                if (i < nops_c) {
                    o = s_opc[i];
                    if (sparse_checks<T>() && s_chk[i]) o.h.x |= OP_CHECK;  // the bound walk's flags (S5)
                    const uint32_t ty = o.h.x & 3u;
                    head = (ty == OP_TT || ty == OP_TTT) && !(o.h.y & TAB_CHECK) && i + 1 < nops_c &&
                           (s_opc[i + 1].h.x & 3u) == OP_SS;
                    if (head) {
                        const OpRec<T> ss = s_opc[i + 1];
                        const uint32_t ss_chk = (!sparse_checks<T>() || s_chk[i + 1]) ? OP_CHECK : 0u;
                        o.h.x = (o.h.x & ~(3u | OP_CHECK | (3u << OP_FUSED_SHIFT))) | OP_TS | ss_chk |
                                ((ty == OP_TTT ? 2u : 1u) << OP_FUSED_SHIFT);
                        o.up[0] = ss.up[0];
                        o.up[1] = ss.up[1];
                    }
                }
                const unsigned mh = __ballot_sync(0xffffffffu, head);
                const bool tail = tid == 0 ? carry : ((mh >> (tid - 1)) & 1u) != 0u;
                const bool keep = i < nops_c && !tail;
                const unsigned mk = __ballot_sync(0xffffffffu, keep);
                const uint32_t j = c_keep + __popc(mk & ((1u << tid) - 1u));
                __syncwarp();
                if (keep) s_opc[j] = o;
                __syncwarp();
                c_keep += __popc(mk);
                carry = (mh >> 31) & 1u;
            }
            if (tid == 0) s_nc = (int)c_keep;
        }
        __syncthreads();
        nops_run = s_nc;
    PTS(6);
    }

    Exact128 ex;
    // the batch loop, instantiated for the unit-diagonal and the standard branch form
    auto batches = [&](auto unit_tag) {
    constexpr bool U = decltype(unit_tag)::value;
    SiteAcc<W> acc;
    Stack<T, DR, SI> st;
    st.sm = smem_addr(s_spill + tid);
#pragma unroll
    for (int k = 0; k < SI; ++k)
#pragma unroll
        for (int i = 0; i < DR; ++i)
#pragma unroll
            for (int j = 0; j < 4; ++j) st.r[k][i][j] = T(0);

    CD cc;
    cc.init(tid);
    const uint32_t s_tab_a = smem_addr(s_tab), s_opc_a = smem_addr(s_opc);
    // exact-sum units of unit_batches batches (the tile starts on a unit boundary); the
    // unit loop keeps the flush out of the batch loop
    for (int b0 = 0; b0 < nb; b0 += a.unit_batches) {
        const int b1 = min(nb, b0 + a.unit_batches);
        for (int b = b0; b < b1; ++b) {
            if (bufs == 2 && b + 1 < nb) {
                issue(b + 1, (b + 1) & 1);
                cp_async_wait<1>();
            } else {  // last batch, or one buffer: this batch's codes were issued before
                cp_async_wait<0>();
            }
            __syncthreads();
            cc.sbase = smem_addr(s_cod + (size_t)(bufs == 2 ? (b & 1) : 0) * bufb);
            int scale[SI];
#pragma unroll
            for (int k = 0; k < SI; ++k) scale[k] = 0;
            uint32_t krow = 0;  // code row of the op's first tip (MPCGS_SLOT_CODES)
            for (int op = 0; op < nops_run; ++op) {
                const uint32_t oa = s_opc_a + (uint32_t)op * (uint32_t)sizeof(OpRec<T>);
                const uint32_t wa = slot_rows<T, GM, DMX, CD>() ? cc.word((int)krow) : 0u;  // issued beside the record load
                const uint4 ox = lds_u4(oa);
                T up[2];
                lds2(up, oa + 16u);
                const UpBr<T, GM, U> ub(up, s_P);
                const int di = (int)((ox.x >> 2) & 15u) * 4 + (int)(ox.x & 3u);  // dense (sp, type) index
                run_op<T, DR, SI, PT, DMX, GM, CD>(di, st, ox.x, ox.y, slot_rows<T, GM, DMX, CD>() ? krow : ox.w,
                                                   slot_rows<T, GM, DMX, CD>() ? wa : cc.word((ox.x >> 6) & 2047), ub, s_tab_a,
                                                   cc, pi, scale);
                krow += op_tips(ox.x);
            }
            const int site0 = s_begin + b * BATCH + tid * SI;
#pragma unroll
            for (int k = 0; k < SI; ++k) {
                T root[4];
                st.template get<0>(k, root);
                T ls = pi[0] * root[0];   // Eq. 21
                ls = fma(pi[1], root[1], ls);
                ls = fma(pi[2], root[2], ls);
                ls = fma(pi[3], root[3], ls);
                if (site0 + k < s_end) acc.add((double)ls, scale[k], a.site_w, site0 + k);  // padding not counted
            }
            __syncthreads();  // the buffer of batch b is refilled in iteration b+1 (one buffer: now)
            if (bufs == 1 && b + 1 < nb) issue(b + 1, 0);
        }
        // this thread's log over the unit (0 if it had no site there)
        ex.add(acc.total());
        acc.reset();
    }
    };
    if constexpr (UK && unit_branch<T, GM>()) {
        if (unit) batches(std::true_type{});
        else batches(std::false_type{});
    } else {
        batches(std::false_type{});
    }
    // the code staging buffers are free now (the last batch ended with a barrier)
    PTS(7);
    exact_commit<PRUNE_THREADS>(ex, a.tree_acc + 4 * (size_t)tree, a.tile_cnt + tree, a.tiles,
                                a.out + (size_t)(a.out_first + tree) * a.out_stride,
                                reinterpret_cast<unsigned long long*>(s_cod), lnC * a.sum_w);
#ifdef MPCGS_PRUNE_TS
    if (threadIdx.x == 0 && blockIdx.x == 0 && blockIdx.y == 0 && (clock64() & 7) == 0)
        printf("prune setup: load %lld compact %lld tables %lld fold %lld fuse %lld | batches %lld (nb %d, ops %d)\n",
               g_pts[2] - g_pts[0], g_pts[3] - g_pts[2], g_pts[4] - g_pts[3], g_pts[5] - g_pts[4], g_pts[6] - g_pts[5],
               g_pts[7] - g_pts[6], nb, nops_run);
#endif
}

template <typename T, int DR, int SI, bool PT, int DMX, bool W, bool GM, int BITS, bool UK>
__global__ void MPCGS_TAB_BOUNDS k_prune_tab(PruneArgs a) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    const int tree = blockIdx.y;
    if (a.tree_need && a.tree_need[tree] > a.need_cap) return;  // deeper tree: scored by the flat pass
    prune_tab_body<T, DR, SI, PT, DMX, W, GM, BITS, UK>(
        a, tree, blockIdx.x, a.sched_op + (size_t)tree * a.nops,
        reinterpret_cast<const typename Traits<T>::E4*>(a.sched_e) + (size_t)tree * a.nops, smem_raw);
}

template <typename T, int D, bool W, bool GM, bool AMB>
static cudaError_t launch_flat_w(const PruneArgs& a, int ntrees, cudaStream_t st) {
    size_t smem = (size_t)a.nops * (sizeof(typename Traits<T>::E4) + sizeof(uint32_t));
    auto kern = k_prune<T, D, W, GM, AMB>;
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

template <typename T, int D, bool GM>
static cudaError_t launch_flat(const PruneArgs& a, int ntrees, cudaStream_t st) {
    if (a.amb)
        return a.site_w ? launch_flat_w<T, D, true, GM, true>(a, ntrees, st)
                        : launch_flat_w<T, D, false, GM, true>(a, ntrees, st);
    return a.site_w ? launch_flat_w<T, D, true, GM, false>(a, ntrees, st)
                    : launch_flat_w<T, D, false, GM, false>(a, ntrees, st);
}

// How many triplets the table kernel may fuse: the shared memory left over at the
// occupancy the kernel reaches without them (registers or base shared memory
// bound it), so fusion never costs a resident CTA.  Cached per tree size; the
// first call is at init (mpcgs_init scores G0), outside any graph capture.
template <typename T, int DR, int SI, bool PT, bool GM, int BITS, typename K>
static int tab_trip_cap(K kern, int nops, int need_cap, int& bufs) {
    // one or two tip-code buffers: one when it buys a resident CTA (cached per tree size)
    static int key[8] = {-1, -1, -1, -1, -1, -1, -1, -1}, val[8], vbufs[8];
    const int k = nops * 16 + need_cap;
    for (int i = 0; i < 8; ++i)
        if (key[i] == k) {
            bufs = vbufs[i];
            return val[i];
        }
    int dev = 0, per_sm = 0, resv = 0, optin = 0, blocks = 0, blocks1 = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&per_sm, cudaDevAttrMaxSharedMemoryPerMultiprocessor, dev);
    cudaDeviceGetAttribute(&resv, cudaDevAttrReservedSharedMemoryPerBlock, dev);
    cudaDeviceGetAttribute(&optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
    int cap = 0;
    bufs = 2;
    size_t base = tab_smem_bytes<T, DR, SI, PT, GM, BITS>(nops, need_cap, 0, 2);
    const size_t base1 = tab_smem_bytes<T, DR, SI, PT, GM, BITS>(nops, need_cap, 0, 1);
    cudaFuncAttributes fa{};
    if (cudaFuncGetAttributes(&fa, kern) == cudaSuccess &&
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, optin - (int)fa.sharedSizeBytes) ==
            cudaSuccess &&
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks, kern, PRUNE_THREADS, base) == cudaSuccess &&
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks1, kern, PRUNE_THREADS, base1) == cudaSuccess) {
        if (MPCGS_SINGLEBUF && blocks1 > blocks) {
            bufs = 1;
            base = base1;
            blocks = blocks1;
        }
        // FP32 general model (96 registers, 5 CTAs/SM by registers): the triplet tables the
        // room at 4 CTAs/SM buys are worth more than the fifth CTA (c5 F84 5.77 -> 5.27 ms,
        // profiles/r02_gm32_occupancy_ab.txt)
        if (GM && sizeof(T) == 4) blocks = std::min(blocks, MPCGS_GM32_MAXCTA);
#ifdef MPCGS_F81_32_MAXCTA  // tuning: the same cap for the FP32 F81 kernel
        if (!GM && sizeof(T) == 4) blocks = std::min(blocks, MPCGS_F81_32_MAXCTA);
#endif
        if (PT && !MPCGS_NO_TRIPLETS && blocks > 0) {
            const long room = std::min<long>(optin, per_sm / blocks - resv - 256) - (long)fa.sharedSizeBytes - (long)base;
            cap = (int)std::max<long>(0, std::min<long>((nops + 1) / 3, room / (long)(sizeof(T) * TRIP_EXTRA)));
        }
    }
    cudaGetLastError();
    for (int i = 0; i < 8; ++i)
        if (key[i] < 0) {
            key[i] = k;
            val[i] = cap;
            vbufs[i] = bufs;
            break;
        }
    return cap;
}

template <typename T, int DR, int SI, bool PT, int DMX, bool W, bool GM, int BITS, bool UK>
static cudaError_t launch_tab_w(PruneArgs a, int ntrees, cudaStream_t st) {
    auto kern = k_prune_tab<T, DR, SI, PT, DMX, W, GM, BITS, UK>;
    a.trip_cap = tab_trip_cap<T, DR, SI, PT, GM, BITS>(kern, a.nops, a.need_cap, a.code_bufs);
    const size_t smem = tab_smem_bytes<T, DR, SI, PT, GM, BITS>(a.nops, a.need_cap, a.trip_cap, a.code_bufs);
    static size_t attr_bytes = 48 * 1024;
    if (smem > attr_bytes) {
        cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        if (e != cudaSuccess) return e;
        attr_bytes = smem;
    }
    dim3 grid(a.tiles, ntrees);
    kern<<<grid, PRUNE_THREADS, smem, st>>>(a);
    return cudaGetLastError();
}

template <typename T, int DR, int SI, bool PT, int DMX, bool GM, int BITS, bool UK>
static cudaError_t launch_tab(const PruneArgs& a, int ntrees, cudaStream_t st) {
    return a.site_w ? launch_tab_w<T, DR, SI, PT, DMX, true, GM, BITS, UK>(a, ntrees, st)
                    : launch_tab_w<T, DR, SI, PT, DMX, false, GM, BITS, UK>(a, ntrees, st);
}

constexpr int PRUNE_SI_LARGE = 2;  // sites per thread for n > 128
#ifndef MPCGS_WIDE_MAX
#define MPCGS_WIDE_MAX 128
#endif
inline bool wide_sites(int n) { return n <= MPCGS_WIDE_MAX; }  // SI sites per thread (else PRUNE_SI_LARGE)
// cherry (16x4) / fused-triplet (64x4) tables: always up to 128 tips; above (with 2 sites
// per thread) only while their shared memory, in the single-code-buffer layout, still
// leaves two CTAs per SM (measured: FP64 n = 192 +12 %, FP32 n = 256 +43 %; FP64 n = 256
// with the round-1 layout needed one CTA per SM and was 20 % slower with tables, with
// the aliased single-buffer layout it fits two and is 4 % faster than without tables at
// three CTAs per SM -- profiles/r02_tables_n256_ab.txt)
#ifndef MPCGS_PT_SMEM_MAX
#define MPCGS_PT_SMEM_MAX (110 * 1024)
#endif
template <typename T, bool GM>
inline bool product_tables(int n) {
    if (n <= 128) return true;
    if (n > 256) return false;
    return tab_smem_bytes<T, PRUNE_DR, PRUNE_SI_LARGE, true, GM>(n - 1, std::min(8, PRUNE_DR + PRUNE_SPILL), 0, 1) <=
           (size_t)MPCGS_PT_SMEM_MAX;
}

template <typename T, int SI, bool PT, bool GM, int BITS = 2, bool UK = false>
static cudaError_t launch_tab_dmx(const PruneArgs& a, int ntrees, cudaStream_t st) {
    switch (a.need_cap) {
        case 1: case 2: case 3: case 4: return launch_tab<T, PRUNE_DR, SI, PT, 4, GM, BITS, UK>(a, ntrees, st);
        case 5: case 6: return launch_tab<T, PRUNE_DR, SI, PT, 6, GM, BITS, UK>(a, ntrees, st);
        case 7: case 8: return launch_tab<T, PRUNE_DR, SI, PT, 8, GM, BITS, UK>(a, ntrees, st);
        default: return launch_tab<T, PRUNE_DR, SI, PT, 10, GM, BITS, UK>(a, ntrees, st);
    }
}

template <typename T, bool GM>
static cudaError_t launch_flat_depth(const PruneArgs& a, int ntrees, int depth, cudaStream_t st) {
    switch (depth) {
        case 4: return launch_flat<T, 4, GM>(a, ntrees, st);
        case 6: return launch_flat<T, 6, GM>(a, ntrees, st);
        case 8: return launch_flat<T, 8, GM>(a, ntrees, st);
        default: return launch_flat<T, 10, GM>(a, ntrees, st);
    }
}

// FP64 F81 table kernels with the unit-diagonal branch loop (prune_f64_unit.cu)
cudaError_t launch_tab_unit_f64(const PruneArgs& a, int ntrees, cudaStream_t st);

// one precision x model: instantiated in prune_{f64,f32}{,_gm}.cu (compiled in parallel)
template <typename T, bool GM>
cudaError_t launch_prune_typed(PruneArgs a, int ntrees, int depth, cudaStream_t st, int& nl) {
    constexpr int SI = sizeof(T) == 4 ? PRUNE_SI32 : PRUNE_SI64;
    const int n = a.nops + 1;
    nl = 0;
    // general model (f4): the flat kernel reads P matrices from sched_P (k_pmat);
    // the table kernel forms its own in shared memory
    auto pmats = [&]() -> cudaError_t {
        if constexpr (!GM) return cudaSuccess;
        const int64_t threads = (int64_t)ntrees * a.nops * 2;
        k_pmat<T><<<(unsigned)((threads + 127) / 128), 128, 0, st>>>(a.sched_e, a.gm, reinterpret_cast<T*>(a.sched_P),
                                                                     a.nops, ntrees);
        ++nl;
        return cudaGetLastError();
    };
    if (a.codes2 == nullptr || !prune_uses_tables(n, sizeof(T) == 4 ? 32 : 64, GM, a.amb != 0)) {
        a.tree_need = nullptr;  // flat kernel for every tree
        cudaError_t e = pmats();
        if (e != cudaSuccess) return e;
        nl += 1;
        return launch_flat_depth<T, GM>(a, ntrees, depth, st);
    }
    a.need_cap = prune_need_cap(n);
    const bool deep = prune_max_need(n) > a.need_cap && a.tree_need != nullptr;
    if (!deep) a.tree_need = nullptr;
    const bool pt = !a.amb && product_tables<T, GM>(n);
    // FP64 F81 on long alignments (a.unit_form): the kernel with the unit-diagonal
    // branch loop, a separate instantiation (prune_f64_unit.cu) -- its second loop
    // instance costs the short-alignment launches 5-9 % (profiles/r02_unit_short_ab.txt)
    const bool unit_kernel = sizeof(T) == 8 && !GM && MPCGS_UNITBR && a.unit_form && !a.amb && pt && wide_sites(n);
    cudaError_t e = unit_kernel ? launch_tab_unit_f64(a, ntrees, st)
                    : a.amb ? (wide_sites(n) ? launch_tab_dmx<T, SI, false, GM, 4>(a, ntrees, st)
                                           : launch_tab_dmx<T, PRUNE_SI_LARGE, false, GM, 4>(a, ntrees, st))
                    : (pt && !wide_sites(n)) ? launch_tab_dmx<T, PRUNE_SI_LARGE, true, GM>(a, ntrees, st)
                    : pt ? launch_tab_dmx<T, SI, true, GM>(a, ntrees, st)
                                      : launch_tab_dmx<T, PRUNE_SI_LARGE, false, GM>(a, ntrees, st);
    nl += 1;
    if (e != cudaSuccess || !deep) return e;
    if ((e = pmats()) != cudaSuccess) return e;
    nl += 1;
    return launch_flat_depth<T, GM>(a, ntrees, depth, st);  // trees with need > cap only
}


extern template cudaError_t launch_prune_typed<double, false>(PruneArgs, int, int, cudaStream_t, int&);
extern template cudaError_t launch_prune_typed<double, true>(PruneArgs, int, int, cudaStream_t, int&);
extern template cudaError_t launch_prune_typed<float, false>(PruneArgs, int, int, cudaStream_t, int&);
extern template cudaError_t launch_prune_typed<float, true>(PruneArgs, int, int, cudaStream_t, int&);

}  // namespace mpcgs

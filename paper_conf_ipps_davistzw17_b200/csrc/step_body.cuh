// step_body.cuh -- device bodies of the GMH step (context, one proposal per warp,
// weights / draws / commit), used by the kernels of step.cu.  Citations as in step.cu.
#pragma once
#include <cfloat>
#include <cstdio>

#include "common.cuh"
#include "kernels.cuh"

namespace mpcgs {

#ifdef MPCGS_TIMESTAMPS
static __device__ long long g_ts[16];
#define MPCGS_TS(i) do { if (threadIdx.x == 0 && blockIdx.x == 0) g_ts[i] = clock64(); } while (0)
static __device__ long long g_tp[8];
#define MPCGS_TP(i) do { if (threadIdx.x == 0 && blockIdx.x == 0) g_tp[i] = clock64(); } while (0)
#else
#define MPCGS_TS(i) do { } while (0)
#define MPCGS_TP(i) do { } while (0)
#endif

constexpr int CTX_THREADS = 256;
// per-interval record of s.omega: [0..8] omega_p(k -> k') at (k-1)*3 + k'-1, [9..11] r1 r2 r3,
// [12] expm1(-(r2-r1) len), [13] expm1(-(r3-r2) len) (the walk's event placement)
constexpr int OM_STRIDE = 16;
constexpr int DRAW_THREADS = 1024;

// ------------------------------------------------------------------ helpers
__device__ __forceinline__ int64_t step_of(const DevState& s, int64_t step_arg) {
    return step_arg >= 0 ? step_arg : s.counters[0];
}

// Scaled weights W^_p(k -> kk) of an interval (length len, l inactive lineages;
// SURVEY App. B closed forms): every weight of the interval carries the common factor
// e^{r_1 len} (S12).
// All six weights of one interval, rows (1,1) (2,2) (2,1) (3,3) (3,2) (3,1), with the
// expressions of what() (the shared exponentials evaluated once).  One thread computes
// a whole row: threads of a warp follow one instruction stream (what() per (interval,
// row) diverged six ways and serialised the transcendentals).
// rt (nullable) receives what the forward walk's event placement needs (OM_STRIDE
// layout): r1, r2, r3 and expm1(-(r2-r1) len), expm1(-(r3-r2) len).
__device__ __forceinline__ void what_row(double len, int l, double theta, bool inf, double* W, double* rt) {
    const double r1 = (2.0 * l) / theta;
    const double r2 = (2.0 + 4.0 * l) / theta;
    const double r3 = (6.0 + 6.0 * l) / theta;
    if (rt) {
        rt[0] = r1; rt[1] = r2; rt[2] = r3;
        rt[3] = inf ? 0.0 : expm1(-(r2 - r1) * len);
        rt[4] = inf ? 0.0 : expm1(-(r3 - r2) * len);
    }
    if (inf) {  // unbounded root interval: only transitions ending at k = 1 (S9)
        W[0] = 1.0; W[1] = 0.0; W[2] = 1.0; W[3] = 0.0; W[4] = 0.0; W[5] = 1.0;
        return;
    }
    const double c2 = 2.0 / theta, c3 = 6.0 / theta;
    const double e21 = exp(-(r2 - r1) * len);
    const double m21 = -expm1(-(r2 - r1) * len);
    const double e31 = exp(-(r3 - r1) * len);
    const double m32 = -expm1(-(r3 - r2) * len);
    const double m31 = -expm1(-(r3 - r1) * len);
    W[0] = 1.0;
    W[1] = e21;
    W[2] = c2 * m21 / (r2 - r1);
    W[3] = e31;
    W[4] = c3 * e21 * m32 / (r3 - r2);
    const double a = m31 / (r3 - r1);
    const double b = e21 * m32 / (r3 - r2);
    W[5] = c3 * c2 * (a - b) / (r2 - r1);
}

// count of x[0..len) <= v (x sorted ascending)
__device__ __forceinline__ int upper_count(const double* x, int len, double v) {
    int lo = 0, hi = len;
    while (lo < hi) {
        int mid = (lo + hi) >> 1;
        if (x[mid] <= v) lo = mid + 1;
        else hi = mid;
    }
    return lo;
}
__device__ __forceinline__ int lower_count(const double* x, int len, double v) {
    int lo = 0, hi = len;
    while (lo < hi) {
        int mid = (lo + hi) >> 1;
        if (x[mid] < v) lo = mid + 1;
        else hi = mid;
    }
    return lo;
}

// exclusive block scan of one int per thread; returns the prefix, total in *tot
template <int NT>
inline __device__ int block_exclusive_scan(int v, int* s_warp, int* tot) {
    const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
    int x = v;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        int y = __shfl_up_sync(0xffffffffu, x, o);
        if (lane >= o) x += y;
    }
    if (lane == 31) s_warp[wid] = x;
    __syncthreads();
    if (wid == 0) {
        int w = lane < NT / 32 ? s_warp[lane] : 0;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            int y = __shfl_up_sync(0xffffffffu, w, o);
            if (lane >= o) w += y;
        }
        if (lane < NT / 32) s_warp[lane] = w;
    }
    __syncthreads();
    int base = wid > 0 ? s_warp[wid - 1] : 0;
    *tot = s_warp[NT / 32 - 1];
    __syncthreads();
    return base + x - v;
}

// ------------------------------------------------------------------ k_context
// Block-wide context computation, NT threads; csm = dynamic shared memory of
// context_smem_bytes(n).  Used by k_context and, for the next step of the
// device loop, at the end of k_draw (saves a launch per step).
template <int NT>
__device__ void context_body(const DevState& s, uint64_t seed, int64_t step_arg, double* csm) {
    MPCGS_TS(5);
    const int n = s.n, nn = s.nn, nint = n - 1;
    double* sAge = csm;               // [n-1] ages of interior nodes (index v - n)
    double* sF = sAge + nint;         // [n] sorted fixed ages
    double* sX = sF + n;              // [n+1] merged cut candidates
    double* sTau = sX + n + 1;        // [n+2]
    double* sW = sTau + n + 2;        // [n][6] W^ rows: (1,1) (2,2) (2,1) (3,3) (3,2) (3,1)
    double* sBeta = sW + 6 * n;       // [(n+1)][3]
    int* sEntry = reinterpret_cast<int*>(sBeta + 3 * (n + 1));  // [n+1]
    int* sPar = sEntry + n + 1;       // [nn] parents, staged: tid 0's lookups below hit shared memory
    int* sLI = sPar + nn;             // [n-1] children of interior nodes (index v - n)
    int* sRI = sLI + nint;            // [n-1]
    __shared__ int sh[16];
    __shared__ double shd[8];
    __shared__ int s_warp[NT / 32];
    const int tid = threadIdx.x;

    for (int i = tid; i < nint; i += NT) {
        sAge[i] = s.age[n + i];
        sLI[i] = s.left[n + i];
        sRI[i] = s.right[n + i];
        if (s.parent[n + i] < 0) sh[10] = n + i;  // root
    }
    for (int i = tid; i < nn; i += NT) sPar[i] = s.parent[i];
    __syncthreads();
    if (tid == 0) {
        const int64_t step = step_of(s, step_arg);
        const int root = sh[10];
        // target: uniform over the n-2 non-root interior nodes in id order (S7)
        U4 w = philox(U4{0u, 0u, (uint32_t)step, TAG_TARGET}, (uint32_t)seed, (uint32_t)(seed >> 32));
        int T = n + (int)__umulhi(w.x, (uint32_t)(n - 2));
        if (T >= root) ++T;
        const int Par = sPar[T];
        const int A = sPar[Par];
        const int sib = sLI[Par - n] == T ? sRI[Par - n] : sLI[Par - n];
        int c[3] = {sLI[T - n], sRI[T - n], sib};
        auto age_of = [&](int v) { return v < n ? 0.0 : sAge[v - n]; };  // tips at age 0 (S22)
        double a[3] = {age_of(c[0]), age_of(c[1]), age_of(c[2])};
        // sort the three children by (age, id)
        for (int i = 0; i < 3; ++i)
            for (int j = i + 1; j < 3; ++j)
                if (a[j] < a[i] || (a[j] == a[i] && c[j] < c[i])) {
                    int tc = c[i]; c[i] = c[j]; c[j] = tc;
                    double ta = a[i]; a[i] = a[j]; a[j] = ta;
                }
        sh[0] = T; sh[1] = Par; sh[2] = A; sh[3] = A < 0; sh[4] = (a[2] == a[1]) ? 3 : 2;
        sh[6] = c[0]; sh[7] = c[1]; sh[8] = c[2];
        shd[0] = a[0]; shd[1] = a[1]; shd[2] = a[2];
        shd[3] = A < 0 ? CUDART_INF : sAge[A - n];
    }
    __syncthreads();
    MPCGS_TS(6);
    const int T = sh[0], Par = sh[1];
    const double a1 = shd[1], a2 = shd[2], tA = shd[3];
    const bool rootcase = sh[3] != 0;
    const int nfixed = n - 3;

    // rank sort of the fixed interior nodes by (age, id)
    for (int v = n + tid; v < nn; v += NT) {
        if (v == T || v == Par) continue;
        const double av = sAge[v - n];
        int r = 0;
        for (int w = n; w < nn; ++w) {
            if (w == T || w == Par) continue;
            const double aw = sAge[w - n];
            r += (aw < av) || (aw == av && w < v);
        }
        sF[r] = av;
    }
    __syncthreads();
    MPCGS_TS(7);
    if (tid == 0) {
        const int lo = upper_count(sF, nfixed, a1);  // fixed ages <= a(2): not cuts
        const int hi = lower_count(sF, nfixed, tA);  // fixed ages <  t_A
        const int has3 = a2 > a1;
        sh[11] = lo;
        sh[12] = hi - lo + has3;                    // merged candidate count
        sh[13] = has3 ? lo + lower_count(sF + lo, hi - lo, a2) - lo : 0;  // insert position
        sh[14] = has3;
    }
    __syncthreads();
    const int lo = sh[11], cnt = sh[12], ins = sh[13], has3 = sh[14];
    for (int j = tid; j < cnt; j += NT) {
        double x;
        if (!has3) x = sF[lo + j];
        else if (j < ins) x = sF[lo + j];
        else if (j == ins) x = a2;
        else x = sF[lo + j - 1];
        sX[j] = x;
    }
    __syncthreads();
    // dedupe (equal ages are one cut) by an exclusive scan of keep flags
    int carry = 0;
    for (int base = 0; base < cnt; base += NT) {
        const int j = base + tid;
        const int keep = (j < cnt) && (j == 0 || sX[j] != sX[j - 1]);
        int tot;
        const int pos = block_exclusive_scan<NT>(keep, s_warp, &tot);
        if (keep) sTau[1 + carry + pos] = sX[j];
        carry += tot;
    }
    const int m = carry + 1;
    if (tid == 0) {
        sTau[0] = a1;
        sTau[m] = tA;
    }
    __syncthreads();
    MPCGS_TS(8);
    // per-interval bookkeeping and closed-form weights: one thread per (interval,
    // weight), 6 weights per interval (the transcendentals dominate)
    for (int p = tid; p < m; p += NT) {
        const double tp = sTau[p];
        const bool inf = rootcase && p == m - 1;
        const double len = inf ? CUDART_INF : sTau[p + 1] - tp;
        const int fixed_below = upper_count(sF, nfixed, tp);
        const int kids_below = (shd[0] <= tp) + (a1 <= tp) + (a2 <= tp);
        const int l = n - fixed_below - kids_below;
        s.tau[p] = tp;
        s.len[p] = len;
        s.lcnt[p] = l;
        sEntry[p] = (p >= 1 && has3 && tp == a2) ? 1 : 0;
        what_row(len, l, s.theta0, inf, sW + p * 6, s.omega + p * OM_STRIDE + 9);  // rows (1,1) (2,2) (2,1) (3,3) (3,2) (3,1)
    }
    if (tid == 0) sEntry[m] = 0;
    __syncthreads();
    MPCGS_TS(9);
    // backward messages (L1005-1020): exactly one lineage at the ancestor
    if (tid == 0) {
        double b1 = 1.0, b2 = 0.0, b3 = 0.0;
        sBeta[m * 3 + 0] = b1; sBeta[m * 3 + 1] = b2; sBeta[m * 3 + 2] = b3;
        for (int p = m - 1; p >= 0; --p) {
            const int en = sEntry[p + 1];
            // beta^end_p(k') = beta_{p+1}(k' + entry_{p+1})
            const double e1 = en ? b2 : b1, e2 = en ? b3 : b2, e3 = en ? 0.0 : b3;
            const double* W = sW + p * 6;
            double n1 = W[0] * e1;
            double n2 = W[1] * e2 + W[2] * e1;
            double n3 = W[3] * e3 + W[4] * e2 + W[5] * e1;
            const double mx = fmax(n1, fmax(n2, n3));
            if (mx > 0.0 && (mx < 0x1p-500 || mx > 0x1p500)) {
                const double f = exp2(-(double)ilogb(mx));   // exact power-of-two rescale
                n1 *= f; n2 *= f; n3 *= f;
            }
            b1 = n1; b2 = n2; b3 = n3;
            sBeta[p * 3 + 0] = b1; sBeta[p * 3 + 1] = b2; sBeta[p * 3 + 2] = b3;
        }
    }
    __syncthreads();
    MPCGS_TS(10);
    // forward choice weights omega_p(k -> k') = W^_p(k -> k') beta_{p+1}(k' + entry_{p+1})
    for (int p = tid; p < m; p += NT) {
        const int en = sEntry[p + 1];
        const double* bn = sBeta + (p + 1) * 3;
        const double be1 = en ? bn[1] : bn[0], be2 = en ? bn[2] : bn[1], be3 = en ? 0.0 : bn[2];
        const double* W = sW + p * 6;
        double* om = s.omega + p * OM_STRIDE;
        om[0] = W[0] * be1; om[1] = 0.0;         om[2] = 0.0;
        om[3] = W[2] * be1; om[4] = W[1] * be2;  om[5] = 0.0;
        om[6] = W[5] * be1; om[7] = W[4] * be2;  om[8] = W[3] * be3;
        s.entry[p] = sEntry[p];
    }
    for (int i = tid; i < nfixed; i += NT) s.fixed[i] = sF[i];
    if (tid == 0) {
        s.tau[m] = tA;
        s.entry[m] = 0;
        for (int i = 0; i < 9; ++i) s.ctx_i[i] = sh[i];
        s.ctx_i[5] = m;
        s.ctx_i[9] = nfixed;
        s.ctx_i[10] = sh[10];
        for (int i = 0; i < 4; ++i) s.ctx_d[i] = shd[i];
        s.counters[4] = T;
        if (s.incremental) {  // ancestors of Par and their other children (f2)
            int d = 0, prev = Par;
            for (int a = sh[2]; a >= 0; a = sPar[a]) {
                s.path[d] = a;
                s.pathsib[d] = sLI[a - n] == prev ? sRI[a - n] : sLI[a - n];
                prev = a;
                ++d;
            }
            s.ctx_i[11] = d;
        }
    }
}


// ------------------------------------------------------------------ k_propose
// One event k -> k-1 in [0, len]: density prop. to e^{-delta s}; inverse CDF with
// em = expm1(-delta len) precomputed by the context (OM_STRIDE record).
__device__ __forceinline__ double place_one_em(double len, double delta, double em, double u, bool inf) {
    if (inf) return -log(u) / delta;
    double sv = -log1p(u * em) / delta;
    return fmin(fmax(sv, 0.0), len);
}

__device__ __forceinline__ double two_cdf(double x, double len, double A, double B) {
    return (-expm1(-(A + B) * x)) / (A + B) - exp(-B * len) * (-expm1(-A * x)) / A;
}

// Two events 3 -> 1 in one interval: joint density e^{-A x - B y} on 0<x<y<len;
// x by safeguarded Newton on its marginal CDF, then y | x by inversion (S13).
inline __device__ void place_two(double len, double A, double B, double u1, double u2, bool inf, double& x,
                          double& y) {
    if (inf) {
        x = -log(u1) / (A + B);
        y = x - log(u2) / B;
        return;
    }
    const double target = u1 * two_cdf(len, len, A, B);
    double lo = 0.0, hi = len;
    // start from the root of the dominant term (exact when e^{-B len} -> 0); the
    // safeguarded iteration then converges to the same root as from len/2 (S13)
    x = -log1p(-u1 * (-expm1(-(A + B) * len))) / (A + B);
    if (!(x > 0.0 && x < len)) x = 0.5 * len;
    // Newton to |dx| <= 2e-14 len (the closed-form CDF cancels when (A+B) len << 1,
    // which bounds its attainable precision), at most 60 iterations
    for (int it = 0; it < 60; ++it) {
        const double f = two_cdf(x, len, A, B) - target;
        const double d = exp(-(A + B) * x) - exp(-B * len - A * x);
        if (f == 0.0) break;
        if (f > 0.0) hi = x;
        else lo = x;
        double xn = (d > 0.0) ? x - f / d : 0.5 * (lo + hi);
        if (fabs(xn - x) <= 2e-14 * len) {  // converged Newton step (checked before the safeguard)
            x = xn;
            break;
        }
        if (!(xn > lo && xn < hi)) xn = 0.5 * (lo + hi);
        x = xn;
    }
    y = x - log1p(u2 * expm1(-B * (len - x))) / B;
    y = fmin(fmax(y, x), len);
}

struct Walk {
    double t1, t2;
    int pair, ok;
};

// Forward walk over the feasible intervals, young -> old (L1028-1034); RNG order
// per interval: choice, event times, then the pair if the first coalescence
// happens with three active lineages.
// int words of k_propose's shared arrays (sL, sR, sNeed, sStack, sLc, sEn, sPar), rounded to even
__host__ __device__ inline int propose_int_words(int n) {
    const int w = 2 * (n - 1) + (2 * n - 1) + 2 * n + (n + 1) + (n + 2) + (2 * n - 1) + 1 + 3 * (n - 1);
    return (w + 1) & ~1;
}

// Warp-parallel emission of exactly the schedule emit_schedule (common.cuh) produces:
// op i of the post-order, code op_encode(type, sp, ta, tb), branch children (ca, cb).
// For an interior node v with subtree size z(v) (interior nodes), first op index s(v)
// and stack depth b(v) when its subtree starts: op index s(v) + z(v) - 1; sp = b(v)
// (TT), b(v) + 1 (TS: after its subtree child), b(v) + 2 (SS).  A child inherits s
// and b, except the second child of an SS node: s + z(first), b + 1 (first = the
// child of larger need, ties to the lower id, as the serial DFS).  Sizes come from
// every interior node walking up to the root (shared atomics), s and b from a second
// walk summing the offsets of the SS nodes passed on the second child's side.
// Returns false (nothing emitted) if some node is deeper than max_walk: the caller
// then runs the serial DFS.
template <typename ET, typename E4, typename EMIT>
__device__ __forceinline__ bool emit_schedule_warp(int n, int lane, const int* sL, const int* sR, const int* sNeed,
                                                   const int* sPar, int* sSize, int max_walk, EMIT emit) {
    const int nn = 2 * n - 1;
    for (int i = lane; i < n - 1; i += 32) sSize[i] = 0;
    __syncwarp();
    bool deep = false;
    for (int u = n + lane; u < nn; u += 32) {
        int k = 0;
        for (int v = u; v >= 0 && k <= max_walk; v = sPar[v], ++k) atomicAdd(sSize + (v - n), 1);
        deep |= k > max_walk;
    }
    if (__any_sync(0xffffffffu, deep)) return false;
    __syncwarp();
    for (int u = n + lane; u < nn; u += 32) {
        int st = 0, bs = 0;
        for (int c = u, p = sPar[u]; p >= 0; c = p, p = sPar[p]) {
            const int a = sL[p - n], b = sR[p - n];
            if (a >= n && b >= n) {
                const int first = sNeed[a] >= sNeed[b] ? a : b;
                if (c != first) {
                    st += sSize[first - n];
                    ++bs;
                }
            }
        }
        const int a = sL[u - n], b = sR[u - n];
        const int idx = st + sSize[u - n] - 1;
        if (a < n && b < n) {
            emit(idx, op_encode(OP_TT, (uint32_t)bs, (uint32_t)a, (uint32_t)b), a, b);
        } else if (a < n || b < n) {
            const int t = a < n ? a : b, w = a < n ? b : a;
            emit(idx, op_encode(OP_TS, (uint32_t)(bs + 1), (uint32_t)t, 0u), t, w);
        } else {
            const int first = sNeed[a] >= sNeed[b] ? a : b, second = first == a ? b : a;
            emit(idx, op_encode(OP_SS, (uint32_t)(bs + 2), 0u, 0u), first, second);
        }
    }
    return true;
}

struct WalkCtx {  // the step's interval context, staged in shared memory
    const double *tau, *len, *omega;
    const int *lcnt, *entry;
    double theta0;
};

// uniforms of the slot's stream: the first PRE_U precomputed by the warp's lanes
constexpr int PRE_U = 64;
struct PreStream {
    const double* pre;
    UStream us;
    __device__ PreStream(const double* p, uint64_t seed, uint32_t slot, uint32_t step)
        : pre(p), us(seed, slot, step, TAG_PROPOSE) {}
    __device__ __forceinline__ double next() {
        const uint32_t i = us.idx;
        if (i < (uint32_t)PRE_U) {
            ++us.idx;
            return pre[i];
        }
        return us.next();
    }
};

inline __device__ Walk forward_walk(const WalkCtx& s, int m, int k0, bool rootcase, uint64_t seed, uint32_t slot,
                             uint32_t step, const double* pre_u) {
    PreStream us(pre_u, seed, slot, step);
    Walk w{0.0, 0.0, 0, 0};
    double tt[2] = {0.0, 0.0};
    int k = k0, events = 0;
    for (int p = 0; p < m && events < 2; ++p) {
        if (p >= 1) k += s.entry[p];
        const bool inf = rootcase && p == m - 1;
        const double* rr = s.omega + p * OM_STRIDE + 9;  // r1 r2 r3 and the expm1 terms (context)
        const double r1 = rr[0], r2 = rr[1], r3 = rr[2];
        const double* om = s.omega + p * OM_STRIDE + (k - 1) * 3;
        const double w0 = om[k - 1];
        const double w1 = k >= 2 ? om[k - 2] : 0.0;
        const double w2 = k >= 3 ? om[k - 3] : 0.0;
        const double u = us.next();
        const double total = (w0 + w1) + w2;
        const double x = u * total;
        int choice;
        double cum = w0;
        if (w0 > 0.0 && cum >= x) choice = 0;
        else {
            cum += w1;
            if (w1 > 0.0 && cum >= x) choice = 1;
            else {
                cum += w2;
                if (w2 > 0.0 && cum >= x) choice = 2;
                else choice = w2 > 0.0 ? 2 : (w1 > 0.0 ? 1 : 0);
            }
        }
        const double len = s.len[p], t0 = s.tau[p];
        if (choice == 1) {
            const double rk = k == 3 ? r3 : (k == 2 ? r2 : r1);
            const double rk1 = k == 3 ? r2 : r1;
            tt[events] = t0 + place_one_em(len, rk - rk1, k == 3 ? rr[4] : rr[3], us.next(), inf);
        } else if (choice == 2) {
            const double u1 = us.next(), u2 = us.next();
            double xo, yo;
            place_two(len, r3 - r2, r2 - r1, u1, u2, inf, xo, yo);
            tt[0] = t0 + xo;
            tt[1] = t0 + yo;
        }
        for (int e = 0; e < choice; ++e) {
            if (events == 0) {
                if (k == 3) {
                    const int pc = (int)(3.0 * us.next());
                    w.pair = pc > 2 ? 2 : pc;
                } else {
                    w.pair = 0;
                }
            }
            ++events;
        }
        k -= choice;
    }
    w.ok = events == 2;
    w.t1 = tt[0];
    w.t2 = tt[1];
    return w;
}

// One warp (lane = threadIdx.x < 32) resimulates proposal `slot` (local index
// `local` of this rank) and emits its register schedule to op_out / e_out (global
// memory for k_prune_tab).
// psm: propose_smem_bytes(n) of shared memory.
template <typename E4, typename ET>
__device__ __forceinline__ void propose_warp(const DevState& s, uint64_t seed, int64_t step_arg, int slot, int local,
                                             int* psm, uint32_t* op_out, E4* e_out) {
    const int n = s.n, nn = s.nn, nint = n - 1;
    // shared copies of the generator and the step context: every sequential
    // lookup of lane 0 (walk, need path, DFS emission) is a shared-memory access
    int* sL = psm;                 // [n-1] children of interior nodes (index v - n)
    int* sR = sL + nint;           // [n-1]
    int* sNeed = sR + nint;        // [nn]
    int* sStack = sNeed + nn;      // [2n]
    int* sLc = sStack + 2 * n;     // [n+1] inactive counts
    int* sEn = sLc + n + 1;        // [n+2] entry flags
    int* sPar = sEn + n + 2;       // [nn] parents
    int* sFlag = sPar + nn;        // [1] serial-emission fallback flag
    int* sSize = sFlag + 1;        // [n-1] subtree sizes for the warp-parallel emission
    double* sTau = reinterpret_cast<double*>(psm + propose_int_words(n));  // [n+2]
    double* sLen = sTau + n + 2;   // [n+1]
    double* sOm = sLen + n + 1;    // [OM_STRIDE (n+1)]
    double* sE = sOm + OM_STRIDE * (n + 1);  // [nn] branch factor above each node (patched for the proposal)
    double* sEm = sE + nn;           // [nn]
    __shared__ double sh_d[8];  // t1, t2, e/em of changed branches
    __shared__ int sh_i[8];
    __shared__ double sU[PRE_U];  // first uniforms of this slot's Philox stream
    const int lane = threadIdx.x;
    MPCGS_TP(0);
    const int64_t step = step_of(s, step_arg);

    const int T = s.ctx_i[0], Par = s.ctx_i[1], A = s.ctx_i[2];
    const bool rootcase = s.ctx_i[3] != 0;
    const int k0 = s.ctx_i[4], m = s.ctx_i[5];
    const int c0 = s.ctx_i[6], c1 = s.ctx_i[7], c2 = s.ctx_i[8];
    const int nfixed = s.ctx_i[9], root = s.ctx_i[10];
    const double ac0 = s.ctx_d[0], ac1 = s.ctx_d[1], ac2 = s.ctx_d[2], tAn = s.ctx_d[3];  // children's / ancestor's ages

    // stage the interval context (L2 reads once, coalesced) for lane 0's sequential walk
    for (int i = lane; i <= m; i += 32) {
        sTau[i] = s.tau[i];
        sEn[i] = s.entry[i];
        if (i < m) {
            sLen[i] = s.len[i];
            sLc[i] = s.lcnt[i];
        }
    }
    for (int i = lane; i < OM_STRIDE * m; i += 32) sOm[i] = s.omega[i];
    for (int i = lane; i < nint; i += 32) {
        sL[i] = s.left[n + i];
        sR[i] = s.right[n + i];
    }
    for (int i = lane; i < nn; i += 32) {
        sNeed[i] = i < n ? 0 : s.need[i];
        sPar[i] = s.parent[i];
        sE[i] = s.e[i];
        sEm[i] = s.em[i];
    }
    MPCGS_TP(1);
    {  // one Philox block per lane: uniforms 2*lane, 2*lane+1 of (slot, step, PROPOSE)
        const U4 b = philox(U4{(uint32_t)lane, (uint32_t)slot, (uint32_t)step, TAG_PROPOSE}, (uint32_t)seed,
                            (uint32_t)(seed >> 32));
        sU[2 * lane] = to_unit(b.x, b.y);
        sU[2 * lane + 1] = to_unit(b.z, b.w);
    }
    __syncwarp();
    if (lane == 0) {
        const WalkCtx wc{sTau, sLen, sOm, sLc, sEn, s.theta0};
        Walk w = forward_walk(wc, m, k0, rootcase, seed, (uint32_t)slot, (uint32_t)step, sU);
        MPCGS_TP(2);
        int pair = w.pair;
        double t1 = w.t1, t2 = w.t2;
        if (!w.ok) {
            // cannot happen for a valid context; keep the generator's tree and flag it
            atomicOr(reinterpret_cast<unsigned long long*>(s.counters + 2), (unsigned long long)STATUS_WALK);
            const int sib = s.left[Par] == T ? s.right[Par] : s.left[Par];
            pair = sib == c2 ? 0 : (sib == c1 ? 1 : 2);
            t1 = s.age[T];
            t2 = s.age[Par];
        }
        sh_i[0] = pair;
        MPCGS_TP(3);
        sh_d[0] = t1;
        sh_d[1] = t2;
    }
    __syncwarp();
    const int pair = sh_i[0];
    const double t1 = sh_d[0], t2 = sh_d[1];
    // pair code 0 = (c1,c2), 1 = (c1,c3), 2 = (c2,c3) (S14)
    const int x = pair == 2 ? c1 : c0;
    const int y = pair == 0 ? c1 : c2;
    const int z = pair == 0 ? c2 : (pair == 1 ? c1 : c0);
    const double u = s.u;
    const double ax = x == c0 ? ac0 : (x == c1 ? ac1 : ac2);
    const double ay = y == c0 ? ac0 : (y == c1 ? ac1 : ac2);
    const double az = z == c0 ? ac0 : (z == c1 ? ac1 : ac2);
    // the five changed branches x, y, z, T, Par: lanes 0..4 evaluate their branch factors
    // in lockstep (one exp + expm1 latency), then lane 0 patches the tree
    __shared__ double sh_e2[4];
    {
        const double lp = rootcase ? 0.0 : tAn - t2;
        const double bt = lane == 0 ? t1 - ax : (lane == 1 ? t1 - ay : (lane == 2 ? t2 - az : (lane == 3 ? t2 - t1 : lp)));
        double be, bem;
        branch_data(s.model, u, bt, be, bem);
        if (lane < 3) {
            sh_d[2 + 2 * lane] = be;
            sh_d[3 + 2 * lane] = bem;
        } else if (lane < 5) {
            sh_e2[2 * (lane - 3)] = be;
            sh_e2[2 * (lane - 3) + 1] = bem;
        }
    }
    if (lane == 0) {
        // younger new node keeps the target's id, older keeps the parent's (S15)
        sL[T - n] = min(x, y);
        sR[T - n] = max(x, y);
        sL[Par - n] = min(T, z);
        sR[Par - n] = max(T, z);
        sNeed[T] = su_need(sNeed[x], sNeed[y]);
        sNeed[Par] = su_need(sNeed[T], sNeed[z]);
        for (int v = A; v >= 0; v = sPar[v]) sNeed[v] = su_need(sNeed[sL[v - n]], sNeed[sR[v - n]]);
        s.tree_need[local] = sNeed[root];
        sPar[x] = T;  // the proposal's parents (Par keeps A)
        sPar[y] = T;
        sPar[z] = Par;
        sPar[T] = Par;
    }
    // S_G of the proposal: merge of the sorted fixed ages with {t1, t2} (Eq. 18 via
    MPCGS_TP(4);
    // S = 2 sum_i (n - i) h_i over sorted coalescence ages)
    double base = 0.0, shift = 0.0;
    int cnt1 = 0, cnt2 = 0;
    for (int q = lane; q < nfixed; q += 32) {
        const double f = s.fixed[q];
        base += (double)(n - (q + 1)) * f;
        shift += (t1 < f ? f : 0.0) + (t2 < f ? f : 0.0);
        cnt1 += f <= t1;
        cnt2 += f <= t2;
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        base += __shfl_xor_sync(0xffffffffu, base, o);
        shift += __shfl_xor_sync(0xffffffffu, shift, o);
        cnt1 += __shfl_xor_sync(0xffffffffu, cnt1, o);
        cnt2 += __shfl_xor_sync(0xffffffffu, cnt2, o);
    }
    __syncwarp();
    if (lane == 0) {
    MPCGS_TP(5);
        const int r1 = 1 + cnt1, r2 = 2 + cnt2;
        const double S = 2.0 * (base - shift) + 2.0 * (double)(n - r1) * t1 + 2.0 * (double)(n - r2) * t2;
        double* rec = s.rec + (size_t)slot * REC;
        rec[1] = S;
        rec[2] = t1;
        rec[3] = t2;
        rec[4] = (double)pair;
        // post-order register schedule of the proposal tree; branch factors of the
        // five changed branches patched into the shared copy
        sE[x] = sh_d[2]; sEm[x] = sh_d[3];
        sE[y] = sh_d[4]; sEm[y] = sh_d[5];
        sE[z] = sh_d[6]; sEm[z] = sh_d[7];
        sE[T] = sh_e2[0]; sEm[T] = sh_e2[1];
        sE[Par] = sh_e2[2]; sEm[Par] = sh_e2[3];
        if (s.incremental) {
            int32_t* q = s.ixyz + 4 * (size_t)local;
            q[0] = x; q[1] = y; q[2] = z; q[3] = 0;
            double* ee = s.iee + 10 * (size_t)local;
            for (int i = 0; i < 6; ++i) ee[i] = sh_d[2 + i];
            for (int i = 0; i < 4; ++i) ee[6 + i] = sh_e2[i];
        }
    }
    __syncwarp();
    // post-order register schedule of the proposal tree (warp-parallel; the serial
    // DFS of emit_schedule for trees deeper than 64 levels)
    auto emit_op = [&](int i, uint32_t code, int ca, int cb) {
        op_out[i] = code;
        E4 v;
        v.x = (ET)sE[ca]; v.y = (ET)sEm[ca]; v.z = (ET)sE[cb]; v.w = (ET)sEm[cb];
        e_out[i] = v;
    };
    const bool par = emit_schedule_warp<ET, E4>(n, lane, sL, sR, sNeed, sPar, sSize, 64, emit_op);
    __syncwarp();
    if (lane == 0) {
        if (!par)
            emit_schedule(
                n, root, [&](int v) { return sL[v - n]; }, [&](int v) { return sR[v - n]; },
                [&](int v) { return sNeed[v]; }, emit_op, sStack);
#ifdef MPCGS_CHECK_SCHED  // verification build: the serial DFS must give the same schedule
        emit_schedule(
            n, root, [&](int v) { return sL[v - n]; }, [&](int v) { return sR[v - n]; },
            [&](int v) { return sNeed[v]; },
            [&](int i, uint32_t code, int ca, int cb) {
                const E4 e = e_out[i];
                if (op_out[i] != code || e.x != (ET)sE[ca] || e.y != (ET)sEm[ca] || e.z != (ET)sE[cb] ||
                    e.w != (ET)sEm[cb])
                    atomicOr(reinterpret_cast<unsigned long long*>(s.counters + 2), (unsigned long long)STATUS_WALK);
            },
            sStack);
#endif
        MPCGS_TP(6);
#ifdef MPCGS_TIMESTAMPS
        if (blockIdx.x == 0 && step == 2)
            printf("propose: stage %lld walk %lld patch %lld e+S %lld pre-dfs %lld dfs %lld\n", g_tp[1] - g_tp[0],
                   g_tp[3] - g_tp[2], g_tp[4] - g_tp[3], g_tp[5] - g_tp[4], g_tp[2] - g_tp[1], g_tp[6] - g_tp[5]);
#endif
    }
}


// ------------------------------------------------------------------ k_draw
// NT threads: 1024, or 128 when N <= 256 (fewer warps at every barrier of a
// latency-bound step; the weights are then a few per thread)
// Records written by other kernels' CTAs are read with ld.global.cg (L2).
__device__ __forceinline__ double rec_ld(const double* p) { return __ldcg(p); }

// Weights, draws, sample store, commit and (loop mode) the next context; NT threads of
// one CTA, dsm = max((N+1) doubles, context_smem_bytes(n)) of shared memory.
template <int NT>
__device__ __forceinline__ void draw_body(const DevState& s, uint64_t seed, int64_t step_arg, int N, int K_arg,
                                          int burnin, int64_t M, int64_t total_steps, double* dsm) {
    MPCGS_TS(0);
    double* sC = dsm;               // [N+1] cumulative weights
    double* sLg = dsm + (N + 1);    // [N+1] logL of every slot, staged once (weights, sample store)
    double* sSg = sLg + (N + 1);    // [N+1] S_G of every slot (sample store)
    __shared__ double s_red[NT / 32];
    __shared__ double s_max;
    __shared__ int s_K, s_store;
    __shared__ long long s_stored;
    const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
    const int64_t step = step_of(s, step_arg);
    const int nslots = N + 1;
    const int T = s.ctx_i[0], Par = s.ctx_i[1];
    if (tid == 0) {
        // slot 0 = the generator with its cached likelihood (S16)
        double* r0 = s.rec;
        r0[0] = s.gen[0];
        r0[1] = s.gen[1];
        r0[2] = s.age[T];
        r0[3] = s.age[Par];
        r0[4] = -1.0;  // read back only after later barriers
    }
    const int chunk = (nslots + NT - 1) / NT;
    const int i0 = tid * chunk, i1 = min(nslots, i0 + chunk);
    const int64_t stored0 = tid == 0 ? s.counters[1] : 0;  // issued early (needed after the barrier)
    double mx = -CUDART_INF;
    for (int i = i0; i < i1; ++i) {
        const double li = i == 0 ? s.gen[0] : rec_ld(s.rec + (size_t)i * REC);
        sLg[i] = li;
        sSg[i] = i == 0 ? s.gen[1] : rec_ld(s.rec + (size_t)i * REC + 1);
        mx = fmax(mx, li);
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) mx = fmax(mx, __shfl_xor_sync(0xffffffffu, mx, o));
    if (lane == 0) s_red[wid] = mx;
    __syncthreads();
    if (tid == 0) {
        double m2 = -CUDART_INF;
        for (int w = 0; w < NT / 32; ++w) m2 = fmax(m2, s_red[w]);
        s_max = m2;
        int K;
        int store;
        if (K_arg >= 0) {
            K = K_arg;
            store = 0;
        } else if (step < burnin) {
            K = 1;  // burn-in: one draw per set, not stored (Fig. 12)
            store = 0;
        } else {
            const int64_t rem = M - stored0;
            K = (int)(rem < N ? rem : N);  // Alg. 1: N draws per set (S17)
            store = 1;
        }
        s_K = K;
        s_store = store;
        s_stored = stored0;
    }
    __syncthreads();
    MPCGS_TS(1);
    mx = s_max;
    if (!(mx > -CUDART_INF) || !(mx < CUDART_INF)) {  // all weights zero or NaN (S6)
        if (tid == 0) {
            atomicOr(reinterpret_cast<unsigned long long*>(s.counters + 2), (unsigned long long)STATUS_NUMERIC);
            if (K_arg < 0) s.counters[0] = step + 1;
        }
        return;
    }
    // w_i = exp(logL_i - max): Eq. 31, proportional to P(D|G_i); inclusive scan in slot order
    double run = 0.0;
    for (int i = i0; i < i1; ++i) {
        run += exp(sLg[i] - mx);
        sC[i] = run;
    }
    double x = run;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        double y = __shfl_up_sync(0xffffffffu, x, o);
        if (lane >= o) x += y;
    }
    __syncthreads();
    if (lane == 31) s_red[wid] = x;
    __syncthreads();
    if (wid == 0) {
        double v = lane < NT / 32 ? s_red[lane] : 0.0;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            double y = __shfl_up_sync(0xffffffffu, v, o);
            if (lane >= o) v += y;
        }
        if (lane < NT / 32) s_red[lane] = v;
    }
    __syncthreads();
    const double before = (wid > 0 ? s_red[wid - 1] : 0.0) + (x - run);
    for (int i = i0; i < i1; ++i) sC[i] += before;
    __syncthreads();
    MPCGS_TS(2);
    const int K = s_K;
    const double total = sC[N];
    const int64_t stored = s_stored;
    for (int d = tid; d < K; d += NT) {
        const double u = uniform_at(seed, 0u, (uint32_t)step, TAG_DRAW, (uint32_t)d);
        const double xd = u * total;
        int lo = 0, hi = N;  // lowest i with C_i >= x (L1140-1144)
        while (lo < hi) {
            const int mid = (lo + hi) >> 1;
            if (sC[mid] >= xd) hi = mid;
            else lo = mid + 1;
        }
        s.last_draws[d] = lo;
        if (s_store) {
            const int64_t j = stored + d;
            s.sS[j] = sSg[lo];
            s.sL[j] = sLg[lo];
            s.sStep[j] = step;
            s.sSlot[j] = lo;
        }
    }
    __syncthreads();
    MPCGS_TS(3);
    // commit: the last draw generates the next proposal set (Fig. 12)
    const int I = K > 0 ? s.last_draws[K - 1] : 0;
    __shared__ double s_be[5], s_bem[5];
    if (I > 0 && tid < 32) {  // the five new branch factors, one lane each, in lockstep
        const double* r = s.rec + (size_t)I * REC;
        const int A = s.ctx_i[2];
        const int c0 = s.ctx_i[6], c1 = s.ctx_i[7], c2 = s.ctx_i[8];
        const int pair = (int)rec_ld(r + 4);
        const double t1 = rec_ld(r + 2), t2 = rec_ld(r + 3);
        const int x = pair == 2 ? c1 : c0;
        const int y = pair == 0 ? c1 : c2;
        const int z = pair == 0 ? c2 : (pair == 1 ? c1 : c0);
        const double lp = A < 0 ? 0.0 : s.age[A] - t2;
        const double bt = tid == 0 ? t1 - s.age[x]
                                   : (tid == 1 ? t1 - s.age[y] : (tid == 2 ? t2 - s.age[z] : (tid == 3 ? t2 - t1 : lp)));
        double be, bem;
        branch_data(s.model, s.u, bt, be, bem);
        if (tid < 5) {
            s_be[tid] = be;
            s_bem[tid] = bem;
        }
    }
    __syncthreads();
    if (tid == 0 && I > 0) {
        const double* r = s.rec + (size_t)I * REC;
        const int A = s.ctx_i[2];
        const int c0 = s.ctx_i[6], c1 = s.ctx_i[7], c2 = s.ctx_i[8];
        const int pair = (int)rec_ld(r + 4);
        const double t1 = rec_ld(r + 2), t2 = rec_ld(r + 3);
        const int x = pair == 2 ? c1 : c0;
        const int y = pair == 0 ? c1 : c2;
        const int z = pair == 0 ? c2 : (pair == 1 ? c1 : c0);
        const int n = s.n;
        s.left[T] = min(x, y);
        s.right[T] = max(x, y);
        s.left[Par] = min(T, z);
        s.right[Par] = max(T, z);
        s.parent[x] = T;
        s.parent[y] = T;
        s.parent[z] = Par;
        s.parent[T] = Par;
        s.age[T] = t1;
        s.age[Par] = t2;
        s.e[x] = s_be[0]; s.em[x] = s_bem[0];
        s.e[y] = s_be[1]; s.em[y] = s_bem[1];
        s.e[z] = s_be[2]; s.em[z] = s_bem[2];
        s.e[T] = s_be[3]; s.em[T] = s_bem[3];
        s.e[Par] = s_be[4]; s.em[Par] = s_bem[4];
        auto nd = [&](int v) { return v < n ? 0 : s.need[v]; };
        s.need[T] = su_need(nd(x), nd(y));
        s.need[Par] = su_need(nd(T), nd(z));
        for (int v = A; v >= 0; v = s.parent[v]) s.need[v] = su_need(nd(s.left[v]), nd(s.right[v]));
        s.gen[0] = rec_ld(r);
        s.gen[1] = rec_ld(r + 1);
    }
    if (tid == 0) {
        if (K_arg < 0) {
            s.counters[0] = step + 1;
            if (s_store) s.counters[1] = stored + K;
        }
        s.counters[3] = K;
    }
    if (tid == 0 && s.incremental) {  // what the partials update (k_commit_incr) needs
        const int d = s.ctx_i[11];
        s.cinfo[0] = T; s.cinfo[1] = Par; s.cinfo[2] = I; s.cinfo[3] = d; s.cinfo[4] = s.ctx_i[3];
        for (int i = 0; i < d; ++i) { s.cpath[i] = s.path[i]; s.csib[i] = s.pathsib[i]; }
    }
    // device loop: the next step's context, from the committed generator
    if (K_arg < 0 && step + 1 < total_steps) {
        __syncthreads();
        MPCGS_TS(4);
        context_body<NT>(s, seed, step + 1, dsm);
        MPCGS_TS(11);
#ifdef MPCGS_TIMESTAMPS
        if (threadIdx.x == 0 && step == 2)
            printf("draw: max %lld scan %lld draws %lld commit %lld | ctx: target %lld sort %lld dedupe %lld W %lld beta %lld rest %lld\n",
                   g_ts[1] - g_ts[0], g_ts[2] - g_ts[1], g_ts[3] - g_ts[2], g_ts[4] - g_ts[3], g_ts[6] - g_ts[5],
                   g_ts[7] - g_ts[6], g_ts[8] - g_ts[7], g_ts[9] - g_ts[8], g_ts[10] - g_ts[9], g_ts[11] - g_ts[10]);
#endif
    }
}


size_t context_smem_bytes(int n);
size_t propose_smem_bytes(int n);

}  // namespace mpcgs

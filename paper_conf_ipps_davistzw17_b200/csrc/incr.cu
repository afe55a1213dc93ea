// incr.cu -- incremental rescoring (the alternative the paper
// weighed and rejected for Kepler, 5.2.2 L1390-1398).
//
// The generator's partial likelihood vector of every interior node at every
// site (Eq. 19) is kept in HBM (GL, with its power-of-two exponent GE).  A
// LAMARC proposal changes only the two resimulated nodes (T, Par) and the
// branch above Par, so its root partial is
//     v_T  = br(L_x) (.) br(L_y),   v_Par = br(v_T) (.) br(L_z),
//     v_a  = br(v_prev) (.) br(L_sib(a))   for a = A, parent(A), ..., root,
// with L_x, L_y, L_z, L_sib(a) read from GL (or tip indicators).  The work per
// proposal and site falls from n-1 nodes to 2 + depth(A) nodes.  After each
// draw k_commit_incr rewrites the changed nodes of the new generator.
// Results equal full pruning up to FP rounding order.
#include <type_traits>

#include "arith.cuh"
#include "common.cuh"
#include "kernels.cuh"

namespace mpcgs {

constexpr int INCR_THREADS = 128;
constexpr int INCR_PG = 8;   // proposals per CTA (per-thread accumulators)
constexpr int INCR_Q = 4;    // proposals whose ancestor chains advance together

// node c at `site`: tip -> indicator vector, exponent 0; interior -> GL, GE
template <typename T>
__device__ __forceinline__ int load_node(const DevState& s, int c, int site, T (&v)[4]) {
    if (c < s.n) {
        const int x = __ldg(s.codes + (size_t)c * s.Lpad + site);
        const int m = s.amb ? x : 1 << x;  // base-set indicator (ambiguity codes: S24)
        v[0] = (m & 1) ? T(1) : T(0);
        v[1] = (m & 2) ? T(1) : T(0);
        v[2] = (m & 4) ? T(1) : T(0);
        v[3] = (m & 8) ? T(1) : T(0);
        return 0;
    }
    const size_t i = (size_t)(c - s.n) * s.Lg + site;
    ld4<T>(v, reinterpret_cast<const T*>(s.GL) + 4 * i);
    return s.GE[i];
}

template <typename T>
__device__ __forceinline__ void store_node(const DevState& s, int v, int site, const T (&x)[4], int e) {
    const size_t i = (size_t)(v - s.n) * s.Lg + site;
    T* g = reinterpret_cast<T*>(s.GL) + 4 * i;
    g[0] = x[0]; g[1] = x[1]; g[2] = x[2]; g[3] = x[3];
    s.GE[i] = e;
}

// v = br(a, ea) (.) br(b, eb), exponent ka + kb (+ own rescale)
template <typename T>
__device__ __forceinline__ int combine(T (&a)[4], int ka, T ea, T ema, T (&b)[4], int kb, T eb, T emb,
                                      const T (&pi)[4]) {
    branch<T>(a, ea, ema, pi);
    branch<T>(b, eb, emb, pi);
#pragma unroll
    for (int i = 0; i < 4; ++i) a[i] *= b[i];
    const int k = rescale_k(a);
    if (k) {
        const T f = pow2(k, T(0));
        a[0] *= f; a[1] *= f; a[2] *= f; a[3] *= f;
    }
    return ka + kb + k;
}

// ---------------------------------------------------------------- full generator partials
template <typename T>
__global__ void __launch_bounds__(256) k_gen_partials(DevState s) {
    const int site = blockIdx.x * blockDim.x + threadIdx.x;
    if (site >= s.L) return;
    const T pi[4] = {(T)s.pi[0], (T)s.pi[1], (T)s.pi[2], (T)s.pi[3]};
    for (int i = 0; i < s.n - 1; ++i) {  // children before parents
        const int v = s.gen_order[i];
        const int l = s.left[v], r = s.right[v];
        T a[4], b[4];
        const int ka = load_node<T>(s, l, site, a);
        const int kb = load_node<T>(s, r, site, b);
        const int k = combine<T>(a, ka, (T)s.e[l], (T)s.em[l], b, kb, (T)s.e[r], (T)s.em[r], pi);
        store_node<T>(s, v, site, a, k);
    }
}

// ---------------------------------------------------------------- commit of the drawn proposal
template <typename T>
__global__ void __launch_bounds__(256) k_commit_incr(DevState s) {
    const int site = blockIdx.x * blockDim.x + threadIdx.x;
    const int I = s.cinfo[2];
    if (I <= 0 || site >= s.L) return;  // the generator was kept: nothing changed
    const T pi[4] = {(T)s.pi[0], (T)s.pi[1], (T)s.pi[2], (T)s.pi[3]};
    const int Tn = s.cinfo[0], Par = s.cinfo[1], d = s.cinfo[3];
    T cur[4], b[4];
    int l = s.left[Tn], r = s.right[Tn];
    int kc = load_node<T>(s, l, site, cur);
    int kb = load_node<T>(s, r, site, b);
    kc = combine<T>(cur, kc, (T)s.e[l], (T)s.em[l], b, kb, (T)s.e[r], (T)s.em[r], pi);
    store_node<T>(s, Tn, site, cur, kc);
    const int z = s.left[Par] == Tn ? s.right[Par] : s.left[Par];
    kb = load_node<T>(s, z, site, b);
    kc = combine<T>(cur, kc, (T)s.e[Tn], (T)s.em[Tn], b, kb, (T)s.e[z], (T)s.em[z], pi);
    store_node<T>(s, Par, site, cur, kc);
    int prev = Par;
    for (int i = 0; i < d; ++i) {
        const int a = s.cpath[i], sib = s.csib[i];
        kb = load_node<T>(s, sib, site, b);
        kc = combine<T>(cur, kc, (T)s.e[prev], (T)s.em[prev], b, kb, (T)s.e[sib], (T)s.em[sib], pi);
        store_node<T>(s, a, site, cur, kc);
        prev = a;
    }
}

// ---------------------------------------------------------------- proposal scores
// Grid (site tiles, ceil(count / INCR_PG)); each CTA scores INCR_PG proposals of
// this rank over one tile.  Per site, the three children's partials and the
// ancestors' sibling factors B_a = br(L_sib(a)) (proposal-independent) are
// computed once -- B_a into shared memory -- and reused by every proposal:
// a proposal then costs two node combines plus one branch and one product per
// ancestor.
constexpr int INCR_DC = 8;  // ancestor levels cached in shared memory per site

template <typename T, bool W>
__global__ void __launch_bounds__(INCR_THREADS) k_score_incr(DevState s, IncrArgs a) {
    __shared__ int sh_sib[128];
    __shared__ double sh_pe[4 * 128];   // e, em of the path branches and of the siblings' branches
    __shared__ int sh_xyz[INCR_PG][4];
    __shared__ double sh_ee[INCR_PG][10];
    using T2 = typename std::conditional<sizeof(T) == 8, double2, float2>::type;
    __shared__ __align__(16) T2 sB[INCR_DC][2][INCR_THREADS];  // B_a of this thread's current site (conflict-free halves)
    __shared__ int sBE[INCR_DC][INCR_THREADS];
    const int tid = threadIdx.x, tile = blockIdx.x;
    const int p0 = blockIdx.y * INCR_PG;
    const int np = min(INCR_PG, a.count - p0);
    const int c0 = s.ctx_i[6], c1 = s.ctx_i[7], c2 = s.ctx_i[8];
    const bool rootcase = s.ctx_i[3] != 0;
    const int d = rootcase ? 0 : s.ctx_i[11];
    const int dc = min(d, 128);  // ancestors whose ids / factors are cached in shared memory
    const int db = min(d, INCR_DC);
    for (int i = tid; i < dc; i += INCR_THREADS) {
        const int an = s.path[i], sb = s.pathsib[i];
        sh_sib[i] = sb;
        sh_pe[4 * i + 0] = s.e[an];
        sh_pe[4 * i + 1] = s.em[an];
        sh_pe[4 * i + 2] = s.e[sb];
        sh_pe[4 * i + 3] = s.em[sb];
    }
    for (int i = tid; i < np * 4; i += INCR_THREADS) sh_xyz[i >> 2][i & 3] = s.ixyz[4 * (p0 + (i >> 2)) + (i & 3)];
    for (int i = tid; i < np * 10; i += INCR_THREADS) sh_ee[i / 10][i % 10] = s.iee[10 * (p0 + i / 10) + i % 10];
    __syncthreads();
    const T pi[4] = {(T)s.pi[0], (T)s.pi[1], (T)s.pi[2], (T)s.pi[3]};
    const int s_begin = tile * a.sites_per_cta;
    const int s_end = min(s.L, s_begin + a.sites_per_cta);
    SiteAcc<W> acc[INCR_PG];
    for (int site = s_begin + tid; site < s_end; site += INCR_THREADS) {
        T L0[4], L1[4], L2[4];
        const int k0 = load_node<T>(s, c0, site, L0);
        const int k1 = load_node<T>(s, c1, site, L1);
        const int k2 = load_node<T>(s, c2, site, L2);
        for (int i = 0; i < db; ++i) {  // B_a, proposal-independent: once per site
            T v[4];
            const int ks = load_node<T>(s, sh_sib[i], site, v);
            branch<T>(v, (T)sh_pe[4 * i + 2], (T)sh_pe[4 * i + 3], pi);
            T2 qa, qb;
            qa.x = v[0]; qa.y = v[1]; qb.x = v[2]; qb.y = v[3];
            sB[i][0][tid] = qa;
            sB[i][1][tid] = qb;
            sBE[i][tid] = ks;
        }
        // INCR_Q proposals advance together: independent chains give the FP pipe ILP
#pragma unroll
        for (int j0 = 0; j0 < INCR_PG; j0 += INCR_Q) {
            if (j0 >= np) break;
            T vx[INCR_Q][4];
            int kc[INCR_Q];
#pragma unroll
            for (int q = 0; q < INCR_Q; ++q) {
                const int j = min(j0 + q, np - 1);  // tail: recompute the last proposal, not stored
                const int x = sh_xyz[j][0], y = sh_xyz[j][1];
                const double* ee = sh_ee[j];
                T vy[4], vz[4];
                int kx, ky, kz;
                // pair code 0 = (c1,c2) | c3, 1 = (c1,c3) | c2, 2 = (c2,c3) | c1 (S14)
                if (x == c0 && y == c1) {
#pragma unroll
                    for (int i = 0; i < 4; ++i) { vx[q][i] = L0[i]; vy[i] = L1[i]; vz[i] = L2[i]; }
                    kx = k0; ky = k1; kz = k2;
                } else if (x == c0) {
#pragma unroll
                    for (int i = 0; i < 4; ++i) { vx[q][i] = L0[i]; vy[i] = L2[i]; vz[i] = L1[i]; }
                    kx = k0; ky = k2; kz = k1;
                } else {
#pragma unroll
                    for (int i = 0; i < 4; ++i) { vx[q][i] = L1[i]; vy[i] = L2[i]; vz[i] = L0[i]; }
                    kx = k1; ky = k2; kz = k0;
                }
                kc[q] = combine<T>(vx[q], kx, (T)ee[0], (T)ee[1], vy, ky, (T)ee[2], (T)ee[3], pi);      // T
                kc[q] = combine<T>(vx[q], kc[q], (T)ee[6], (T)ee[7], vz, kz, (T)ee[4], (T)ee[5], pi);   // Par
            }
            for (int i = 0; i < d; ++i) {
                T bs[4];
                int ks;
                if (i < db) {
                    const T2 qa = sB[i][0][tid], qb = sB[i][1][tid];
                    bs[0] = qa.x; bs[1] = qa.y; bs[2] = qb.x; bs[3] = qb.y;
                    ks = sBE[i][tid];
                } else {  // deep paths: recompute the sibling factor
                    const int sb = i < dc ? sh_sib[i] : s.pathsib[i];
                    ks = load_node<T>(s, sb, site, bs);
                    branch<T>(bs, (T)s.e[sb], (T)s.em[sb], pi);
                }
#pragma unroll
                for (int q = 0; q < INCR_Q; ++q) {
                    const int j = min(j0 + q, np - 1);
                    T pe, pem;  // branch from the previous path node: Par -> A, then a(i-1) -> a(i)
                    if (i == 0) { pe = (T)sh_ee[j][8]; pem = (T)sh_ee[j][9]; }
                    else if (i - 1 < dc) { pe = (T)sh_pe[4 * (i - 1) + 0]; pem = (T)sh_pe[4 * (i - 1) + 1]; }
                    else { const int an = s.path[i - 1]; pe = (T)s.e[an]; pem = (T)s.em[an]; }
                    branch<T>(vx[q], pe, pem, pi);
#pragma unroll
                    for (int r = 0; r < 4; ++r) vx[q][r] *= bs[r];
                    const int kr = rescale_k(vx[q]);
                    if (kr) {
                        const T f = pow2(kr, T(0));
                        vx[q][0] *= f; vx[q][1] *= f; vx[q][2] *= f; vx[q][3] *= f;
                    }
                    kc[q] += ks + kr;
                }
            }
#pragma unroll
            for (int q = 0; q < INCR_Q; ++q) {
                const int j = j0 + q;
                if (j >= np) break;
                // Eq. 21 at the root, multiplied into this proposal's accumulator
                T ls = pi[0] * vx[q][0];
                ls = fma(pi[1], vx[q][1], ls);
                ls = fma(pi[2], vx[q][2], ls);
                ls = fma(pi[3], vx[q][3], ls);
                acc[j].add((double)ls, kc[q], s.site_w, site);
            }
        }
    }
    // per proposal: this thread's log over the tile, summed exactly (arith.cuh Exact128)
    __shared__ ExactScratch<INCR_THREADS> s_ex;
#pragma unroll
    for (int j = 0; j < INCR_PG; ++j) {
        if (j >= np) break;  // np is uniform in the CTA
        Exact128 ex;
        ex.add(acc[j].total());
        const int tree = p0 + j;
        exact_commit<INCR_THREADS>(ex, a.tree_acc + 4 * (size_t)tree, a.tile_cnt + tree, a.tiles,
                                   a.out + (size_t)(a.out_first + tree) * a.out_stride, s_ex.w);
    }
}

cudaError_t launch_gen_partials(const DevState& s, cudaStream_t st) {
    const int blocks = (s.L + 255) / 256;
    if (s.precision == 32) k_gen_partials<float><<<blocks, 256, 0, st>>>(s);
    else k_gen_partials<double><<<blocks, 256, 0, st>>>(s);
    return cudaGetLastError();
}

cudaError_t launch_commit_incr(const DevState& s, cudaStream_t st) {
    const int blocks = (s.L + 255) / 256;
    if (s.precision == 32) k_commit_incr<float><<<blocks, 256, 0, st>>>(s);
    else k_commit_incr<double><<<blocks, 256, 0, st>>>(s);
    return cudaGetLastError();
}

cudaError_t launch_score_incr(const DevState& s, const IncrArgs& a, cudaStream_t st) {
    if (a.count <= 0) return cudaSuccess;
    dim3 grid(a.tiles, (a.count + INCR_PG - 1) / INCR_PG);
    const bool w = s.site_w != nullptr;
    if (s.precision == 32) {
        if (w) k_score_incr<float, true><<<grid, INCR_THREADS, 0, st>>>(s, a);
        else k_score_incr<float, false><<<grid, INCR_THREADS, 0, st>>>(s, a);
    } else {
        if (w) k_score_incr<double, true><<<grid, INCR_THREADS, 0, st>>>(s, a);
        else k_score_incr<double, false><<<grid, INCR_THREADS, 0, st>>>(s, a);
    }
    return cudaGetLastError();
}

}  // namespace mpcgs

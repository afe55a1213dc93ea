// common.cuh -- device state layout, Philox4x32-10, schedule encoding.
//
// Product code of the B200 mpcgs library (no oracle code is included or
// shared).  Citations "L<a>-<b>" refer to PAPER.md (Davis 2016); readings
// S1..S23 to DESIGN.md.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>
#include <math_constants.h>

namespace mpcgs {

constexpr uint32_t TAG_TARGET = 0u;   // counter tag of the target-node draw (4.3, S7)
constexpr uint32_t TAG_PROPOSE = 1u;  // per-proposal resimulation stream (4.2)
constexpr uint32_t TAG_DRAW = 2u;     // inverse-CDF draws of the step (L1140-1144)

constexpr int REC = 5;  // record per slot: logL, S, t1, t2, pair

// ---------------------------------------------------------------- Philox4x32-10
// Counter-based generator (Salmon et al. 2011) replacing MT19937/MTGP32
// (5.1.2 L1243-1256): counter (block, slot or draw group, step, tag), key = seed.
struct U4 {
    uint32_t x, y, z, w;
};

__host__ __device__ __forceinline__ void mulhilo32(uint32_t a, uint32_t b, uint32_t& hi, uint32_t& lo) {
#ifdef __CUDA_ARCH__
    hi = __umulhi(a, b);
    lo = a * b;
#else
    uint64_t p = (uint64_t)a * (uint64_t)b;
    hi = (uint32_t)(p >> 32);
    lo = (uint32_t)p;
#endif
}

__host__ __device__ __forceinline__ U4 philox(U4 c, uint32_t k0, uint32_t k1) {
#pragma unroll
    for (int r = 0; r < 10; ++r) {
        uint32_t hi0, lo0, hi1, lo1;
        mulhilo32(0xD2511F53u, c.x, hi0, lo0);
        mulhilo32(0xCD9E8D57u, c.z, hi1, lo1);
        U4 o;
        o.x = hi1 ^ c.y ^ k0;
        o.y = lo1;
        o.z = hi0 ^ c.w ^ k1;
        o.w = lo0;
        c = o;
        k0 += 0x9E3779B9u;
        k1 += 0xBB67AE85u;
    }
    return c;
}

// 53 random bits + one ulp: exactly representable, in (0, 1].
__host__ __device__ __forceinline__ double to_unit(uint32_t a, uint32_t b) {
    return ((double)(a >> 5) * 67108864.0 + (double)(b >> 6) + 1.0) * (1.0 / 9007199254740992.0);
}

// Sequential uniforms of one stream (c1, step, tag); two doubles per Philox block.
struct UStream {
    uint32_t k0, k1, c1, step, tag, idx;
    U4 blk;
    __host__ __device__ UStream(uint64_t seed, uint32_t c1_, uint32_t step_, uint32_t tag_)
        : k0((uint32_t)seed), k1((uint32_t)(seed >> 32)), c1(c1_), step(step_), tag(tag_), idx(0) {}
    __host__ __device__ double next() {
        if ((idx & 1u) == 0u) blk = philox(U4{idx >> 1, c1, step, tag}, k0, k1);
        double u = (idx & 1u) ? to_unit(blk.z, blk.w) : to_unit(blk.x, blk.y);
        ++idx;
        return u;
    }
};

__host__ __device__ __forceinline__ double uniform_at(uint64_t seed, uint32_t c1, uint32_t step, uint32_t tag,
                                                      uint32_t idx) {
    U4 b = philox(U4{idx >> 1, c1, step, tag}, (uint32_t)seed, (uint32_t)(seed >> 32));
    return (idx & 1u) ? to_unit(b.z, b.w) : to_unit(b.x, b.y);
}

// ---------------------------------------------------------------- schedule encoding
// One op per interior node, children before parents (Sethi-Ullman order), on a
// register stack R[0..D): bits 0-1 type, 2-5 sp (stack depth before the op),
// 6-16 tip a, 17-27 tip b.
//   TT (type 0): R[sp]   = tip(a) (.) tip(b)                     sp -> sp+1
//   TS (type 1): R[sp-1] = tip(a) (.) branch(R[sp-1])            sp unchanged
//   SS (type 2): R[sp-2] = branch(R[sp-2]) (.) branch(R[sp-1])   sp -> sp-1
// Branch data per op: {e_a, em_a, e_b, em_b}, e = exp(-u t), em = -expm1(-u t)
// (Eq. 20: P_XY(t) = e delta_XY + em pi_Y).  For TS, (e_a, em_a) belong to the
// tip and (e_b, em_b) to the stack child.
constexpr uint32_t OP_TT = 0u, OP_TS = 1u, OP_SS = 2u;
__host__ __device__ __forceinline__ uint32_t op_encode(uint32_t type, uint32_t sp, uint32_t ta, uint32_t tb) {
    return type | (sp << 2) | (ta << 6) | (tb << 17);
}

__host__ __device__ __forceinline__ int su_need(int a, int b) { return a == b ? a + 1 : (a > b ? a : b); }

// Emit the post-order register schedule of a tree.  Generic over array access so
// that the host (score_trees, G0) and the propose kernel (smem) share it.
//   kidL(v), kidR(v): children of interior node v (ids, lower first)
//   need(v): Sethi-Ullman register need (tips 0)
//   emit(i, code, ca, cb): op i with branch children ca (tip a / first) and cb
// Returns the maximum stack depth.  stack: scratch of >= 2n entries.
template <class KL, class KR, class NEED, class EMIT>
__host__ __device__ int emit_schedule(int n, int root, KL kidL, KR kidR, NEED need, EMIT emit, int* stack) {
    int top = 0, sp = 0, nop = 0, maxsp = 0;
    stack[top++] = root << 2;
    while (top > 0) {
        int fr = stack[top - 1];
        int v = fr >> 2, st = fr & 3;
        int a = kidL(v), b = kidR(v);
        if (st == 0) {
            if (a < n && b < n) {
                emit(nop++, op_encode(OP_TT, sp, a, b), a, b);
                ++sp;
                if (sp > maxsp) maxsp = sp;
                --top;
            } else if (a < n || b < n) {
                int w = a < n ? b : a;
                stack[top - 1] = (v << 2) | 3;
                stack[top++] = w << 2;
            } else {
                int first = need(a) >= need(b) ? a : b;
                stack[top - 1] = (v << 2) | 1;
                stack[top++] = first << 2;
            }
        } else if (st == 3) {
            int t = a < n ? a : b, w = a < n ? b : a;
            emit(nop++, op_encode(OP_TS, sp, t, 0), t, w);
            --top;
        } else if (st == 1) {
            int second = need(a) >= need(b) ? b : a;
            stack[top - 1] = (v << 2) | 2;
            stack[top++] = second << 2;
        } else {
            int first = need(a) >= need(b) ? a : b, second = first == a ? b : a;
            emit(nop++, op_encode(OP_SS, sp, 0, 0), first, second);
            --sp;
            --top;
        }
    }
    return maxsp;
}

// ---------------------------------------------------------------- device state
struct DevState {
    int n, nn, L, Lpad, nops, precision;
    double pi[4];
    double u;       // F81 rate (S3)
    double theta0;  // driving value
    int model;             // 0: F81 (Eq. 20), branch data e/em.  1: general reversible model
                           // (F84, HKY85: SURVEY 8(f) f4), branch data (t, 0), P(t) from gm
    const double* gm;      // [36] ev[4], V[16], W[16]: P(t) = V diag(exp(ev t)) W (model 1)
    void* sched_P;         // [Nmax][nops][32] P of each op's two children (model 1)
    int amb;               // 1: codes are base-set masks 1..15 (ambiguity codes, f4 / S24)
    const uint8_t* codes;  // [n][Lpad], 0..3 (or masks when amb)
    const double* site_w;  // [L] pattern counts when sites are compressed patterns (f3), else nullptr
    // generator (chain state)
    int32_t *parent, *left, *right, *need;  // [nn] (left/right/need valid for interior)
    double *age, *e, *em;                   // [nn]; e/em of the branch above each node
    double* gen;                            // [0] logL, [1] S
    // per-step context (4.2 L986-1027)
    int32_t* ctx_i;    // T, Par, A, rootcase, k0, m, c0, c1, c2, nfixed
    double* ctx_d;     // a0, a1, a2, tA
    double* tau;       // [n+1]
    double* len;       // [n]
    int32_t* lcnt;     // [n]
    int32_t* entry;    // [n+1]
    double* omega;     // [n+1][16]: omega_p(k -> k') at (k-1)*3 + k'-1, then r1 r2 r3, expm1 terms
    double* fixed;     // [n] sorted ages of interior nodes other than T, Par
    // proposals
    double* rec;        // [(Nmax+1)][REC]
    int32_t* tree_need; // [Nmax] register need of each local proposal's schedule
    uint32_t* sched_op; // [Nmax][nops]
    void* sched_e;      // [Nmax][nops] x {e_a, em_a, e_b, em_b} (float or double)
    unsigned long long* tree_acc;  // [Nmax][4] exact site-sum accumulators (arith.cuh Exact128)
    uint32_t* tile_cnt; // [Nmax]
    // samples (5.1.3 L1264-1269: S_G suffices for Eq. 18)
    double *sS, *sL;
    int64_t* sStep;
    int32_t* sSlot;
    int64_t* counters;  // [0] step, [1] stored, [2] status, [3] last K, [4] last target
    int32_t* last_draws;
    double* theta_buf;
    int Nmax, tiles_max;
    int64_t Mmax;
    // incremental rescoring: the generator's partial likelihood
    // of every interior node at every site, and what each proposal changed
    int incremental;
    void* GL;           // [n-1][Lg][4] partials of interior node v at [v-n] (float or double)
    int32_t* GE;        // [n-1][Lg] power-of-two exponent removed from GL (whole subtree)
    int Lg;             // site stride of GL / GE
    int32_t* path;      // [n] ancestors of Par: A, parent(A), ..., root (context)
    int32_t* pathsib;   // [n] the other child of each ancestor
    int32_t* ixyz;      // [Nmax][4] per local proposal: pair children x, y and third child z
    double* iee;        // [Nmax][10] e/em of the changed branches x, y, z, T, Par
    int32_t* cinfo;     // committed step: T, Par, I (drawn slot), d, rootcase
    int32_t* cpath;     // [n] committed step's ancestor path
    int32_t* csib;      // [n]
    int32_t* gen_order; // [n-1] interior nodes children-first (full partial recompute)
};

// Transition matrix of a general reversible model from its eigen-decomposition
// gm = {ev[4], V[16], W[16]}: P_ij(t) = sum_k V_ik exp(ev_k t) W_kj (row i = the
// state at the parent end).  Entries are clamped at 0 (true P(t) >= 0; the
// eigen route leaves rounding-size negatives near t = 0).
__host__ __device__ inline void pmat(const double* gm, double t, double* P) {
    double ex[4];
    for (int k = 0; k < 4; ++k) ex[k] = exp(gm[k] * t);
    for (int i = 0; i < 4; ++i)
        for (int j = 0; j < 4; ++j) {
            double v = 0.0;
            for (int k = 0; k < 4; ++k) v = fma(gm[4 + i * 4 + k] * ex[k], gm[20 + k * 4 + j], v);
            P[i * 4 + j] = v > 0.0 ? v : 0.0;
        }
}

// Branch data of a branch of length t: F81 {e, em} = {exp(-u t), -expm1(-u t)}
// (Eq. 20); general model {t, 0} (P(t) is formed per op by k_pmat).
__host__ __device__ __forceinline__ void branch_data(int model, double u, double t, double& e, double& em) {
    if (model) {
        e = t;
        em = 0.0;
    } else {
        e = exp(-u * t);
        em = -expm1(-u * t);
    }
}

// counters[2] status bits
constexpr int64_t STATUS_NUMERIC = 1;
constexpr int64_t STATUS_WALK = 2;

}  // namespace mpcgs

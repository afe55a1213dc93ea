/*
 * oracle.c -- plain FP64 CPU oracle of the mpcgs hot path.
 *
 * TEST INFRASTRUCTURE ONLY (see oracle.h).  Scalar C99, no SIMD, no threads,
 * no code shared with the CUDA library.  Written for a reader checking it
 * against PAPER.md by eye, not for speed.
 *
 * Parity status of each function:
 *   philox / u01 ........ pinned: Random123 known-answer vectors (P17)
 *   F81 transition ...... pinned: rows sum to 1, P(0)=I, P(inf)=1 pi^T, Chapman-Kolmogorov (P1)
 *   log_likelihood ...... pinned: brute-force ancestral enumeration n=2..5 (P3), pulley (P4/P5),
 *                          permutation/duplication (P6), zero branches (P7), monomorphic (P2)
 *   coalescent_S / prior  pinned: S identity, E[T_k] (P10), closed form Eq. 18
 *   pick_target ......... pinned: uniform over n-2 non-root interior nodes (chi-square)
 *   context / propose ... pinned: interval-event probabilities vs 2-D quadrature of the
 *                          restricted prior (P13), n=3 prior law (P12), n=4 topology law (P11)
 *   weights / draw ...... pinned: softmax invariance and prior cancellation (P14, P15)
 *   gmh_step / chain .... pinned: n=3 exact posterior by quadrature (P16), prior chain (P11)
 *   MLE ................. pinned: M=1 closed form, bracket, stationarity, EM monotone,
 *                          bimodal global mode (P18)
 *   upgma ............... pinned: hand-worked 4-taxon example
 */
#include "oracle.h"

#include <math.h>
#include <stdlib.h>
#include <string.h>

/* ------------------------------------------------------------------------- */
/* RNG: Philox4x32-10 (Salmon et al. 2011, Random123).  Replaces the paper's   */
/* host MT19937 + device MTGP32 (5.1.2 L1243-1256), reading S21.               */
/* Counter = (block index within the stream, slot or draw group, step, tag),  */
/* key = (seed low 32 bits, seed high 32 bits).                                */
/* ------------------------------------------------------------------------- */
void orc_philox4x32_10(const uint32_t ctr[4], const uint32_t key[2], uint32_t out[4]) {
    uint32_t x0 = ctr[0], x1 = ctr[1], x2 = ctr[2], x3 = ctr[3];
    uint32_t k0 = key[0], k1 = key[1];
    int round;
    for (round = 0; round < 10; ++round) {
        uint64_t prod0, prod1;
        uint32_t hi0, lo0, hi1, lo1;
        if (round > 0) {          /* key schedule: bump by the Weyl constants */
            k0 += 0x9E3779B9u;
            k1 += 0xBB67AE85u;
        }
        prod0 = (uint64_t)0xD2511F53u * (uint64_t)x0;
        prod1 = (uint64_t)0xCD9E8D57u * (uint64_t)x2;
        hi0 = (uint32_t)(prod0 >> 32);
        lo0 = (uint32_t)prod0;
        hi1 = (uint32_t)(prod1 >> 32);
        lo1 = (uint32_t)prod1;
        x0 = hi1 ^ x1 ^ k0;
        x1 = lo1;
        x2 = hi0 ^ x3 ^ k1;
        x3 = lo0;
    }
    out[0] = x0;
    out[1] = x1;
    out[2] = x2;
    out[3] = x3;
}

/* Two 32-bit words -> a double in (0, 1]: 53 random bits, plus one ulp. */
double orc_u01(uint32_t w0, uint32_t w1) {
    double hi = (double)(w0 >> 5);   /* 27 bits */
    double lo = (double)(w1 >> 6);   /* 26 bits */
    return (hi * 67108864.0 + lo + 1.0) * (1.0 / 9007199254740992.0);
}

/* The idx-th uniform of stream (c1, step, tag): block idx/2, words 2*(idx%2)..+1 */
double orc_uniform(uint64_t seed, uint32_t c1, uint32_t step, uint32_t tag, uint32_t idx) {
    uint32_t ctr[4], key[2], out[4];
    ctr[0] = idx / 2u;
    ctr[1] = c1;
    ctr[2] = step;
    ctr[3] = tag;
    key[0] = (uint32_t)(seed & 0xFFFFFFFFu);
    key[1] = (uint32_t)(seed >> 32);
    orc_philox4x32_10(ctr, key, out);
    if (idx % 2u == 0u) return orc_u01(out[0], out[1]);
    return orc_u01(out[2], out[3]);
}

/* ------------------------------------------------------------------------- */
/* F81 model.                                                                 */
/* ------------------------------------------------------------------------- */

/* pi_Y = relative frequency of nucleotide Y over all n*L characters (L702-703, S1). */
void orc_base_freqs(int n, int L, const uint8_t* codes, double pi[4]) {
    double count[4] = {0.0, 0.0, 0.0, 0.0};
    long i, total = (long)n * (long)L;
    int X;
    double known = 0.0;
    /* ambiguity codes (>= 16, S24) are not counted */
    for (i = 0; i < total; ++i)
        if (codes[i] < 4) {
            count[codes[i]] += 1.0;
            known += 1.0;
        }
    for (X = 0; X < 4; ++X) pi[X] = known > 0 ? count[X] / known : 0.25;
}

/* u = 1 / (1 - sum pi^2) so that branch lengths are expected substitutions (S3). */
double orc_default_rate(const double pi[4]) {
    double s = pi[0] * pi[0] + pi[1] * pi[1] + pi[2] * pi[2] + pi[3] * pi[3];
    if (s >= 1.0) return 1.0;
    return 1.0 / (1.0 - s);
}

/* Eq. 20 (L696-699): P_XY(t) = e^{-ut} delta_XY + (1 - e^{-ut}) pi_Y.  P[X*4+Y]. */
void orc_transition(double t, double u, const double pi[4], double P[16]) {
    double stay = exp(-u * t);
    int X, Y;
    for (X = 0; X < 4; ++X)
        for (Y = 0; Y < 4; ++Y) P[X * 4 + Y] = (X == Y ? stay : 0.0) + (1.0 - stay) * pi[Y];
}

/* purine/pyrimidine group of a state and the group's total frequency */
static int group_of(int X) { return (X == 0 || X == 2) ? 0 : 1; }
static double group_freq(int X, const double pi[4]) {
    return group_of(X) == 0 ? pi[0] + pi[2] : pi[1] + pi[3];
}

/* Rate mu that makes the expected number of substitutions per unit time 1. */
double orc_model_rate(int model, double kappa, const double pi[4]) {
    double sum = 0.0;
    int X, Y;
    if (model == 0) return orc_default_rate(pi);
    for (X = 0; X < 4; ++X)
        for (Y = 0; Y < 4; ++Y) {
            double q;
            if (X == Y) continue;
            if (model == 1) /* F84: pi_Y (1 + kappa / Pi_g [same group]) */
                q = pi[Y] * (1.0 + (group_of(X) == group_of(Y) ? kappa / group_freq(Y, pi) : 0.0));
            else /* HKY85: kappa pi_Y for transitions, pi_Y for transversions */
                q = (group_of(X) == group_of(Y) ? kappa : 1.0) * pi[Y];
            sum += pi[X] * q;
        }
    return sum > 0.0 ? 1.0 / sum : 1.0;
}

void orc_transition_model(int model, double kappa, double t, const double pi[4], double P[16]) {
    double mu = orc_model_rate(model, kappa, pi);
    int X, Y;
    if (model == 0) {
        orc_transition(t, mu, pi, P);
        return;
    }
    for (X = 0; X < 4; ++X)
        for (Y = 0; Y < 4; ++Y) {
            double PiY = group_freq(Y, pi), v;
            int same = group_of(X) == group_of(Y);
            if (model == 1) {
                /* F84 (Felsenstein 1984): e^{-(1+k)mu t} d_XY
                   + e^{-mu t}(1 - e^{-k mu t}) pi_Y / Pi_Y [same group] + (1 - e^{-mu t}) pi_Y */
                v = (X == Y ? exp(-(1.0 + kappa) * mu * t) : 0.0) +
                    (same ? exp(-mu * t) * (1.0 - exp(-kappa * mu * t)) * pi[Y] / PiY : 0.0) +
                    (1.0 - exp(-mu * t)) * pi[Y];
            } else {
                /* HKY85 (Hasegawa, Kishino & Yano 1985), A_Y = 1 + Pi_Y (kappa - 1) */
                double A = 1.0 + PiY * (kappa - 1.0);
                if (X == Y)
                    v = pi[Y] + pi[Y] * (1.0 / PiY - 1.0) * exp(-mu * t) + ((PiY - pi[Y]) / PiY) * exp(-mu * A * t);
                else if (same)
                    v = pi[Y] + pi[Y] * (1.0 / PiY - 1.0) * exp(-mu * t) - (pi[Y] / PiY) * exp(-mu * A * t);
                else
                    v = pi[Y] * (1.0 - exp(-mu * t));
            }
            P[X * 4 + Y] = v;
        }
}

/* ------------------------------------------------------------------------- */
/* Tree helpers.                                                              */
/* ------------------------------------------------------------------------- */
static void children_of(int n, const int32_t* parent, int32_t* left, int32_t* right) {
    int nn = 2 * n - 1, v;
    for (v = 0; v < nn; ++v) {
        left[v] = -1;
        right[v] = -1;
    }
    for (v = 0; v < nn; ++v) {            /* ascending v: left child gets the lower id */
        int p = parent[v];
        if (p < 0) continue;
        if (left[p] < 0) left[p] = v;
        else right[p] = v;
    }
}

static int root_of(int n, const int32_t* parent) {
    int v;
    for (v = 0; v < 2 * n - 1; ++v)
        if (parent[v] < 0) return v;
    return -1;
}

int orc_check_tree(int n, const int32_t* parent, const double* age) {
    int nn = 2 * n - 1, v, roots = 0;
    int* nchild;
    if (n < 2) return ORC_E_ARG;
    nchild = (int*)calloc((size_t)nn, sizeof(int));
    for (v = 0; v < nn; ++v) {
        int p = parent[v];
        if (p < 0) {
            roots++;
            continue;
        }
        if (p < n || p >= nn || p == v) {
            free(nchild);
            return ORC_E_TREE;
        }
        nchild[p]++;
        if (!(age[p] >= age[v])) {
            free(nchild);
            return ORC_E_TREE;
        }
    }
    for (v = 0; v < nn; ++v) {
        if (v < n && nchild[v] != 0) roots = -100;
        if (v >= n && nchild[v] != 2) roots = -100;
    }
    free(nchild);
    if (roots != 1) return ORC_E_TREE;
    if (parent[root_of(n, parent)] != -1) return ORC_E_TREE;
    if (root_of(n, parent) < n) return ORC_E_TREE;
    return ORC_OK;
}

/* ------------------------------------------------------------------------- */
/* Data likelihood (Felsenstein pruning, Eq. 19-22) in log space (5.3).        */
/* ------------------------------------------------------------------------- */

/* Eq. 32 generalised to m terms: ln sum e^{x_i} = k + ln sum e^{x_i - k}, k = max. */
static double log_sum_exp(const double* x, int m) {
    double k = -INFINITY, s = 0.0;
    int i;
    for (i = 0; i < m; ++i)
        if (x[i] > k) k = x[i];
    if (k == -INFINITY) return -INFINITY;
    for (i = 0; i < m; ++i) s += exp(x[i] - k);
    return k + log(s);
}

typedef struct {
    int n, L;
    const uint8_t* codes;
    const int32_t* left;
    const int32_t* right;
    const double* lnP;   /* per child node v: ln P(age[parent v] - age[v]), 16 entries */
    double* lnL;         /* per node, 4 entries: ln L_v(X) at the current site */
} prune_work;

/* Post-order recursion (2.4 L685-690): fills ln L_v(X) for the current site. */
static void prune_node(prune_work* w, int v, int site) {
    double* out = w->lnL + 4 * v;
    int X, Y, side;
    if (v < w->n) {
        /* Tips are indicator vectors (L673-676): L = 1 for the observed base; an
           ambiguity code (16 + set, reading S24) is the indicator
           of its set of bases (Felsenstein 1981, 2004 ch. 16). */
        int code = w->codes[(long)v * w->L + site];
        int set = code < 4 ? 1 << code : code - 16;
        for (X = 0; X < 4; ++X) out[X] = ((set >> X) & 1) ? 0.0 : -INFINITY;
        return;
    }
    for (X = 0; X < 4; ++X) out[X] = 0.0;
    for (side = 0; side < 2; ++side) {
        int c = side == 0 ? w->left[v] : w->right[v];
        const double* lnPc = w->lnP + 16 * c;
        const double* lnLc;
        prune_node(w, c, site);
        lnLc = w->lnL + 4 * c;
        /* Eq. 19: L_v(X) = prod_children sum_Y P_XY(t_vc) L_c(Y), each sum in log space */
        for (X = 0; X < 4; ++X) {
            double terms[4];
            for (Y = 0; Y < 4; ++Y) terms[Y] = lnPc[X * 4 + Y] + lnLc[Y];
            out[X] += log_sum_exp(terms, 4);
        }
    }
}

static double log_likelihood_impl(int model, double kappa, double u, int n, int L, const uint8_t* codes,
                                  const int32_t* parent, const double* age, const double pi[4],
                                  double* site_ll);

double orc_log_likelihood(int n, int L, const uint8_t* codes, const int32_t* parent,
                          const double* age, const double pi[4], double u, double* site_ll) {
    return log_likelihood_impl(0, 0.0, u, n, L, codes, parent, age, pi, site_ll);
}

double orc_log_likelihood_model(int model, double kappa, int n, int L, const uint8_t* codes,
                                const int32_t* parent, const double* age, const double pi[4],
                                double* site_ll) {
    return log_likelihood_impl(model, kappa, 0.0, n, L, codes, parent, age, pi, site_ll);
}

static double log_likelihood_impl(int model, double kappa, double u, int n, int L, const uint8_t* codes,
                                  const int32_t* parent, const double* age, const double pi[4],
                                  double* site_ll) {
    int nn = 2 * n - 1, v, s, X;
    int32_t* left = (int32_t*)malloc(sizeof(int32_t) * (size_t)nn);
    int32_t* right = (int32_t*)malloc(sizeof(int32_t) * (size_t)nn);
    double* lnP = (double*)malloc(sizeof(double) * 16 * (size_t)nn);
    double* lnL = (double*)malloc(sizeof(double) * 4 * (size_t)nn);
    double sum = 0.0, comp = 0.0;   /* Neumaier compensated sum over sites */
    int root = root_of(n, parent);
    prune_work w;
    children_of(n, parent, left, right);
    for (v = 0; v < nn; ++v) {
        double P[16];
        int i;
        if (parent[v] < 0) continue;
        if (model == 0) orc_transition(age[parent[v]] - age[v], u, pi, P);
        else orc_transition_model(model, kappa, age[parent[v]] - age[v], pi, P);
        for (i = 0; i < 16; ++i) lnP[16 * v + i] = log(P[i]);
    }
    w.n = n;
    w.L = L;
    w.codes = codes;
    w.left = left;
    w.right = right;
    w.lnP = lnP;
    w.lnL = lnL;
    for (s = 0; s < L; ++s) {
        double terms[4], ell, t;
        prune_node(&w, root, s);
        /* Eq. 21: L_s(G) = sum_X pi_X L_root(X) */
        for (X = 0; X < 4; ++X) terms[X] = log(pi[X]) + lnL[4 * root + X];
        ell = log_sum_exp(terms, 4);
        if (site_ll) site_ll[s] = ell;
        /* Eq. 22 read as a product over independent sites (S4): sum of logs */
        if (ell == -INFINITY) {
            sum = -INFINITY;
            comp = 0.0;
            continue;
        }
        if (sum == -INFINITY) continue;
        t = sum + ell;
        if (fabs(sum) >= fabs(ell)) comp += (sum - t) + ell;
        else comp += (ell - t) + sum;
        sum = t;
    }
    free(left);
    free(right);
    free(lnP);
    free(lnL);
    if (sum == -INFINITY) return -INFINITY;
    return sum + comp;
}

/* ------------------------------------------------------------------------- */
/* Coalescent prior, Eq. 17-18 (reading S8).                                  */
/* ------------------------------------------------------------------------- */
static int cmp_double(const void* a, const void* b) {
    double x = *(const double*)a, y = *(const double*)b;
    return (x > y) - (x < y);
}

/* S_G = sum_{k=2}^{n} k(k-1) T_k, T_k = length of the interval with k lineages. */
double orc_coalescent_S(int n, const double* age) {
    double* h = (double*)malloc(sizeof(double) * (size_t)(n - 1));
    double S = 0.0, prev = 0.0;
    int i, k;
    for (i = 0; i < n - 1; ++i) h[i] = age[n + i];
    qsort(h, (size_t)(n - 1), sizeof(double), cmp_double);
    /* between the (i)-th and (i+1)-th coalescence (ages h[i-1], h[i]) there are n-i lineages */
    for (i = 0; i < n - 1; ++i) {
        k = n - i;
        S += (double)k * (double)(k - 1) * (h[i] - prev);
        prev = h[i];
    }
    free(h);
    return S;
}

/* Eq. 18: ln P(G|theta) = (n-1) ln(2/theta) - S_G / theta. */
double orc_log_prior(int n, const double* age, double theta) {
    return (double)(n - 1) * log(2.0 / theta) - orc_coalescent_S(n, age) / theta;
}

/* ------------------------------------------------------------------------- */
/* Target node (4.3 L1079-1093; S7): uniform over the n-2 non-root interior   */
/* nodes in ascending id order, from one Philox word (Lemire multiply-shift).  */
/* ------------------------------------------------------------------------- */
int orc_pick_target(int n, const int32_t* parent, uint64_t seed, uint32_t step) {
    uint32_t ctr[4] = {0u, 0u, step, ORC_TAG_TARGET};
    uint32_t key[2], out[4];
    uint32_t idx;
    int v, seen = 0;
    key[0] = (uint32_t)(seed & 0xFFFFFFFFu);
    key[1] = (uint32_t)(seed >> 32);
    orc_philox4x32_10(ctr, key, out);
    idx = (uint32_t)(((uint64_t)out[0] * (uint64_t)(n - 2)) >> 32);
    for (v = n; v < 2 * n - 1; ++v) {
        if (parent[v] < 0) continue;
        if ((uint32_t)seen == idx) return v;
        seen++;
    }
    return -1;
}

/* ------------------------------------------------------------------------- */
/* Neighbourhood context (4.2 L986-1027), readings S9-S12.                    */
/* ------------------------------------------------------------------------- */
typedef struct {
    int T, Par, A, rootcase;
    int c[3];
    double a[3];
    int k0, m;
    double theta;
    double* tau;    /* m+1 boundaries, tau[m] = age(A) or +inf */
    double* len;    /* m interval lengths */
    int* l;         /* m inactive-lineage counts */
    int* entry;     /* m+1 flags: third child enters at the start of interval p */
    double* What;   /* m*9 scaled transition weights W^_p(k -> k') at [(k-1)*3 + k'-1] */
    double* beta;   /* (m+1)*3 backward messages (the paper's P_i(n), L1017-1020) */
} orc_ctx;

static void ctx_free(orc_ctx* c) {
    free(c->tau);
    free(c->len);
    free(c->l);
    free(c->entry);
    free(c->What);
    free(c->beta);
}

/*
 * Weight of starting an interval of length `len` with k active lineages and
 * ending it with kk, when l inactive lineages are present (S10/S12):
 * active pairs coalesce at 2/theta each; active-inactive coalescences are
 * forbidden (killed at 2kl/theta).  r_k = (k(k-1) + 2kl)/theta is the exit
 * rate, c_k = k(k-1)/theta the coalescence prefactor.  Every weight of the
 * interval is multiplied by the common factor e^{r_1 len}; a common factor
 * per interval does not change any conditional choice (Appendix B).
 */
static double What_k(int k, int kk, double len, int l, double theta, int infinite) {
    double r1 = (2.0 * l) / theta;
    double r2 = (2.0 + 4.0 * l) / theta;
    double r3 = (6.0 + 6.0 * l) / theta;
    double c2 = 2.0 / theta, c3 = 6.0 / theta;
    if (infinite) {
        /* unbounded root interval, l = 0: every lineage must coalesce (S9) */
        return kk == 1 ? 1.0 : 0.0;
    }
    if (k == 1 && kk == 1) return 1.0;
    if (k == 2 && kk == 2) return exp(-(r2 - r1) * len);
    if (k == 2 && kk == 1) return c2 * (-expm1(-(r2 - r1) * len)) / (r2 - r1);
    if (k == 3 && kk == 3) return exp(-(r3 - r1) * len);
    if (k == 3 && kk == 2)
        return c3 * exp(-(r2 - r1) * len) * (-expm1(-(r3 - r2) * len)) / (r3 - r2);
    if (k == 3 && kk == 1) {
        double first = (-expm1(-(r3 - r1) * len)) / (r3 - r1);
        double second = exp(-(r2 - r1) * len) * (-expm1(-(r3 - r2) * len)) / (r3 - r2);
        return c3 * c2 * (first - second) / (r2 - r1);
    }
    return 0.0;
}

static int build_context(int n, const int32_t* parent, const double* age, double theta0,
                         int target, orc_ctx* cx) {
    int nn = 2 * n - 1;
    int32_t* left = (int32_t*)malloc(sizeof(int32_t) * (size_t)nn);
    int32_t* right = (int32_t*)malloc(sizeof(int32_t) * (size_t)nn);
    double* cuts = (double*)malloc(sizeof(double) * (size_t)(n + 2));
    int ncut = 0, nuniq, v, i, j, p, k;
    double tA;
    memset(cx, 0, sizeof(*cx));
    if (target < n || target >= nn || parent[target] < 0) {
        free(left);
        free(right);
        free(cuts);
        return ORC_E_ARG;
    }
    children_of(n, parent, left, right);
    cx->theta = theta0;
    cx->T = target;
    cx->Par = parent[target];
    cx->A = parent[cx->Par];
    cx->rootcase = cx->A < 0;
    /* children of the neighbourhood: both children of T and T's sibling (L986-995) */
    cx->c[0] = left[target];
    cx->c[1] = right[target];
    cx->c[2] = left[cx->Par] == target ? right[cx->Par] : left[cx->Par];
    /* sort by (age, id) */
    for (i = 0; i < 3; ++i)
        for (j = i + 1; j < 3; ++j) {
            int ci = cx->c[i], cj = cx->c[j];
            if (age[cj] < age[ci] || (age[cj] == age[ci] && cj < ci)) {
                cx->c[i] = cj;
                cx->c[j] = ci;
            }
        }
    for (i = 0; i < 3; ++i) cx->a[i] = age[cx->c[i]];
    tA = cx->rootcase ? INFINITY : age[cx->A];
    /* backward time (S11): the region starts at the second child's age a(2) */
    cx->k0 = (cx->a[2] == cx->a[1]) ? 3 : 2;
    if (cx->a[2] > cx->a[1]) cuts[ncut++] = cx->a[2];
    for (v = n; v < nn; ++v) {
        if (v == cx->T || v == cx->Par) continue;
        if (age[v] > cx->a[1] && age[v] < tA) cuts[ncut++] = age[v];
    }
    qsort(cuts, (size_t)ncut, sizeof(double), cmp_double);
    nuniq = 0;
    for (i = 0; i < ncut; ++i)
        if (nuniq == 0 || cuts[i] != cuts[nuniq - 1]) cuts[nuniq++] = cuts[i];
    cx->m = nuniq + 1;
    cx->tau = (double*)malloc(sizeof(double) * (size_t)(cx->m + 1));
    cx->len = (double*)malloc(sizeof(double) * (size_t)cx->m);
    cx->l = (int*)malloc(sizeof(int) * (size_t)cx->m);
    cx->entry = (int*)calloc((size_t)(cx->m + 1), sizeof(int));
    cx->What = (double*)calloc((size_t)cx->m * 9, sizeof(double));
    cx->beta = (double*)calloc((size_t)(cx->m + 1) * 3, sizeof(double));
    cx->tau[0] = cx->a[1];
    for (i = 0; i < nuniq; ++i) cx->tau[i + 1] = cuts[i];
    cx->tau[cx->m] = tA;
    for (p = 0; p < cx->m; ++p) {
        int fixed_below = 0, kids_below = 0;
        double tp = cx->tau[p];
        cx->len[p] = cx->tau[p + 1] - tp;
        /* inactive lineages: all lineages of the pruned tree at tau_p minus active ones */
        for (v = n; v < nn; ++v)
            if (v != cx->T && v != cx->Par && age[v] <= tp) fixed_below++;
        for (i = 0; i < 3; ++i)
            if (cx->a[i] <= tp) kids_below++;
        cx->l[p] = n - fixed_below - kids_below;
        if (p >= 1 && cx->a[2] > cx->a[1] && tp == cx->a[2]) cx->entry[p] = 1;
    }
    for (p = 0; p < cx->m; ++p) {
        int inf = (p == cx->m - 1) && cx->rootcase;
        for (k = 1; k <= 3; ++k) {
            int kk;
            for (kk = 1; kk <= k; ++kk)
                cx->What[p * 9 + (k - 1) * 3 + (kk - 1)] =
                    What_k(k, kk, cx->len[p], cx->l[p], theta0, inf);
        }
    }
    /* Backward recursion for P_i(n) (L1005-1020): exactly one lineage at the ancestor */
    cx->beta[cx->m * 3 + 0] = 1.0;
    for (p = cx->m - 1; p >= 0; --p) {
        double mx = 0.0;
        for (k = 1; k <= 3; ++k) {
            double s = 0.0;
            int kk;
            for (kk = (k - 2 > 1 ? k - 2 : 1); kk <= k; ++kk) {
                int ke = kk + cx->entry[p + 1];
                double be = ke <= 3 ? cx->beta[(p + 1) * 3 + (ke - 1)] : 0.0;
                s += cx->What[p * 9 + (k - 1) * 3 + (kk - 1)] * be;
            }
            cx->beta[p * 3 + (k - 1)] = s;
            if (s > mx) mx = s;
        }
        if (mx > 0.0)
            for (k = 0; k < 3; ++k) cx->beta[p * 3 + k] /= mx;   /* keep the scale O(1) */
    }
    free(left);
    free(right);
    free(cuts);
    return ORC_OK;
}

/* omega_p(k -> kk) = W^_p(k -> kk) * beta_{p+1}(kk + entry_{p+1}): forward choice weight */
static double omega(const orc_ctx* cx, int p, int k, int kk) {
    int ke = kk + cx->entry[p + 1];
    double be;
    if (kk < 1 || kk > k) return 0.0;
    be = ke <= 3 ? cx->beta[(p + 1) * 3 + (ke - 1)] : 0.0;
    return cx->What[p * 9 + (k - 1) * 3 + (kk - 1)] * be;
}

int orc_context_info(int n, const int32_t* parent, const double* age, double theta0, int target,
                     int32_t* info, double* tau, double* len, int32_t* l, int32_t* entry,
                     double* om, double* beta) {
    orc_ctx cx;
    int rc = build_context(n, parent, age, theta0, target, &cx), p, k, kk;
    if (rc != ORC_OK) return rc;
    info[0] = cx.T;
    info[1] = cx.Par;
    info[2] = cx.A;
    info[3] = cx.rootcase;
    info[4] = cx.k0;
    info[5] = cx.m;
    info[6] = cx.c[0];
    info[7] = cx.c[1];
    info[8] = cx.c[2];
    for (p = 0; p <= cx.m; ++p) {
        if (tau) tau[p] = cx.tau[p];
        if (entry) entry[p] = cx.entry[p];
        if (beta)
            for (k = 0; k < 3; ++k) beta[p * 3 + k] = cx.beta[p * 3 + k];
    }
    for (p = 0; p < cx.m; ++p) {
        if (len) len[p] = cx.len[p];
        if (l) l[p] = cx.l[p];
        if (om)
            for (k = 1; k <= 3; ++k)
                for (kk = 1; kk <= 3; ++kk) om[p * 9 + (k - 1) * 3 + (kk - 1)] = omega(&cx, p, k, kk);
    }
    ctx_free(&cx);
    return ORC_OK;
}

/* ------------------------------------------------------------------------- */
/* Resimulation (4.2 L1028-1043) with the RNG order of SURVEY 8(c) c7:         */
/* per interval walked: 1 choice uniform; then the event-time uniforms of that */
/* interval; then the pair uniform if the proposal's first coalescence fell in */
/* this interval with three active lineages.  The walk stops after the second  */
/* coalescence.                                                               */
/* ------------------------------------------------------------------------- */
typedef struct {
    uint64_t seed;
    uint32_t slot, step, idx;
} ustream;

static double next_u(ustream* s) {
    return orc_uniform(s->seed, s->slot, s->step, ORC_TAG_PROPOSE, s->idx++);
}

#define NEAR_TOL 1e-9

/* lowest index whose cumulative weight reaches x = u * total (L1140-1144) */
static int choose(const double* wts, int m, double u, int* flag) {
    double total = 0.0, cum = 0.0, x;
    int i;
    for (i = 0; i < m; ++i) total += wts[i];
    x = u * total;
    for (i = 0; i < m; ++i) {
        cum += wts[i];
        if (wts[i] > 0.0 && fabs(cum - x) <= NEAR_TOL * total) *flag = 1;
        if (cum >= x && wts[i] > 0.0) return i;
    }
    for (i = m - 1; i >= 0; --i)
        if (wts[i] > 0.0) return i;
    return 0;
}

/* One event k -> k-1 in [0, len]: density prop. to e^{-delta s} (Appendix B), inverse CDF */
static double place_one(double len, double delta, double u, int infinite) {
    double s;
    if (infinite) return -log(u) / delta;
    s = -log1p(u * expm1(-delta * len)) / delta;
    if (s > len) s = len;
    if (s < 0.0) s = 0.0;
    return s;
}

/* Unnormalised CDF of the first of two events: joint density e^{-A x - B y}, 0<x<y<len */
static double two_event_cdf(double x, double len, double A, double B) {
    return (-expm1(-(A + B) * x)) / (A + B) - exp(-B * len) * (-expm1(-A * x)) / A;
}

/* Two events 3 -> 1 in one interval (S13): x by safeguarded Newton inversion, then y | x */
static void place_two(double len, double A, double B, double u1, double u2, int infinite,
                      double* x_out, double* y_out) {
    double x, y;
    if (infinite) {
        x = -log(u1) / (A + B);
        y = x - log(u2) / B;
    } else {
        double target = u1 * two_event_cdf(len, len, A, B);
        double lo = 0.0, hi = len;
        int it;
        x = 0.5 * len;
        for (it = 0; it < 100; ++it) {
            double f = two_event_cdf(x, len, A, B) - target;
            double d = exp(-(A + B) * x) - exp(-B * len - A * x);
            double xn;
            if (f > 0.0) hi = x;
            else lo = x;
            xn = (d > 0.0) ? x - f / d : 0.5 * (lo + hi);
            if (!(xn > lo && xn < hi)) xn = 0.5 * (lo + hi);
            if (fabs(xn - x) <= 1e-15 * len) {
                x = xn;
                break;
            }
            x = xn;
        }
        y = x - log1p(u2 * expm1(-B * (len - x))) / B;
        if (y > len) y = len;
        if (y < x) y = x;
    }
    *x_out = x;
    *y_out = y;
}

static int propose_from_ctx(int n, const int32_t* parent, const double* age, const orc_ctx* cx,
                            uint64_t seed, uint32_t step, uint32_t slot, int32_t* new_parent,
                            double* new_age, double* t12, int32_t* pair_out, int32_t* flag) {
    ustream us;
    int k = cx->k0, p, events = 0, pair = 0, nn = 2 * n - 1, v;
    double times[2] = {0.0, 0.0};
    int x_child, y_child, z_child;
    *flag = 0;
    us.seed = seed;
    us.slot = slot;
    us.step = step;
    us.idx = 0;
    for (p = 0; p < cx->m && events < 2; ++p) {
        double wts[3], u;
        int choice, kk, ne, e;
        int inf = (p == cx->m - 1) && cx->rootcase;
        double theta = cx->theta;
        double r[4];
        if (p >= 1) k += cx->entry[p];
        r[1] = (2.0 * cx->l[p]) / theta;
        r[2] = (2.0 + 4.0 * cx->l[p]) / theta;
        r[3] = (6.0 + 6.0 * cx->l[p]) / theta;
        /* forward walk (L1028-1034): choose the end state in order k, k-1, k-2 */
        wts[0] = omega(cx, p, k, k);
        wts[1] = omega(cx, p, k, k - 1);
        wts[2] = omega(cx, p, k, k - 2);
        u = next_u(&us);
        choice = choose(wts, 3, u, flag);
        kk = k - choice;
        ne = k - kk;
        if (ne == 1) {
            double s = place_one(cx->len[p], r[k] - r[k - 1], next_u(&us), inf);
            times[events] = cx->tau[p] + s;
        } else if (ne == 2) {
            double u1 = next_u(&us), u2 = next_u(&us), xo, yo;
            place_two(cx->len[p], r[3] - r[2], r[2] - r[1], u1, u2, inf, &xo, &yo);
            times[0] = cx->tau[p] + xo;
            times[1] = cx->tau[p] + yo;
        }
        for (e = 0; e < ne; ++e) {
            if (events == 0) {
                /* first coalescence: with three active lineages the pair is uniform (S14) */
                if (k == 3) {
                    double up = next_u(&us);
                    double f = 3.0 * up;
                    pair = (int)f;
                    if (pair > 2) pair = 2;
                    if (fabs(f - 1.0) <= 3.0 * NEAR_TOL || fabs(f - 2.0) <= 3.0 * NEAR_TOL) *flag = 1;
                } else {
                    pair = 0;
                }
            }
            events++;
        }
        k = kk;
    }
    if (events != 2) return ORC_E_NUMERIC;
    /* pair code: 0 = (c1,c2), 1 = (c1,c3), 2 = (c2,c3) */
    if (pair == 0) {
        x_child = cx->c[0];
        y_child = cx->c[1];
        z_child = cx->c[2];
    } else if (pair == 1) {
        x_child = cx->c[0];
        y_child = cx->c[2];
        z_child = cx->c[1];
    } else {
        x_child = cx->c[1];
        y_child = cx->c[2];
        z_child = cx->c[0];
    }
    for (v = 0; v < nn; ++v) {
        new_parent[v] = parent[v];
        new_age[v] = age[v];
    }
    /* younger new node keeps the target's id, older keeps the parent's id (S15) */
    new_parent[x_child] = cx->T;
    new_parent[y_child] = cx->T;
    new_parent[z_child] = cx->Par;
    new_parent[cx->T] = cx->Par;
    new_parent[cx->Par] = cx->rootcase ? -1 : cx->A;
    new_age[cx->T] = times[0];
    new_age[cx->Par] = times[1];
    t12[0] = times[0];
    t12[1] = times[1];
    *pair_out = pair;
    return ORC_OK;
}

int orc_propose(int n, const int32_t* parent, const double* age, double theta0, int target,
                uint64_t seed, uint32_t step, uint32_t slot, int32_t* new_parent,
                double* new_age, double* t12, int32_t* pair, int32_t* flag) {
    orc_ctx cx;
    int rc = build_context(n, parent, age, theta0, target, &cx);
    if (rc != ORC_OK) return rc;
    rc = propose_from_ctx(n, parent, age, &cx, seed, step, slot, new_parent, new_age, t12, pair,
                          flag);
    ctx_free(&cx);
    return rc;
}

/* ------------------------------------------------------------------------- */
/* Weights and draws.  Eq. 29-31: pi_i K(G_i, G_\i) is proportional to         */
/* P(D|G_i) -- the prior cancels (S18), so the weights are softmax(logL).      */
/* ------------------------------------------------------------------------- */
int orc_weights(int nslots, const double* logL, double* w, double* cum) {
    double mx = -INFINITY, run = 0.0;
    int i;
    for (i = 0; i < nslots; ++i)
        if (logL[i] > mx) mx = logL[i];
    if (!(mx > -INFINITY) || !isfinite(mx)) return ORC_E_NUMERIC;
    for (i = 0; i < nslots; ++i) {
        w[i] = exp(logL[i] - mx);
        run += w[i];
        cum[i] = run;
    }
    return ORC_OK;
}

/* x = u * sum w; I = lowest j with cumulative >= x (L1140-1144) */
int orc_draw(int nslots, const double* cum, double u, int32_t* flag) {
    double total = cum[nslots - 1], x = u * total;
    int i;
    *flag = 0;
    for (i = 0; i < nslots; ++i) {
        if (fabs(cum[i] - x) <= NEAR_TOL * total) *flag = 1;
        if (cum[i] >= x) return i;
    }
    return nslots - 1;
}

static int gmh_step_impl(int model, double kappa, int n, int L, const uint8_t* codes,
                         const double pi[4], double u, double theta0, int N, int K, uint64_t seed,
                         uint32_t step, int32_t* gen_parent, double* gen_age, double* gen_logL,
                         int32_t* out_target, double* slot_logL, double* slot_S, double* slot_t12,
                         int32_t* slot_pair, int32_t* slot_flag, int32_t* draws, int32_t* draw_flag) {
    int nn = 2 * n - 1, i, d, rc, last = 0;
    int32_t* par_all = (int32_t*)malloc(sizeof(int32_t) * (size_t)nn * (size_t)(N + 1));
    double* age_all = (double*)malloc(sizeof(double) * (size_t)nn * (size_t)(N + 1));
    double* w = (double*)malloc(sizeof(double) * (size_t)(N + 1));
    double* cum = (double*)malloc(sizeof(double) * (size_t)(N + 1));
    orc_ctx cx;
    int target = orc_pick_target(n, gen_parent, seed, step);
    *out_target = target;
    rc = build_context(n, gen_parent, gen_age, theta0, target, &cx);
    if (rc != ORC_OK) goto done;
    /* slot 0 = the generator, whose likelihood is cached (S16) */
    memcpy(par_all, gen_parent, sizeof(int32_t) * (size_t)nn);
    memcpy(age_all, gen_age, sizeof(double) * (size_t)nn);
    slot_logL[0] = *gen_logL;
    slot_S[0] = orc_coalescent_S(n, gen_age);
    slot_t12[0] = gen_age[target];
    slot_t12[1] = gen_age[gen_parent[target]];
    slot_pair[0] = -1;
    slot_flag[0] = 0;
    for (i = 1; i <= N; ++i) {
        int32_t* pp = par_all + (size_t)i * nn;
        double* aa = age_all + (size_t)i * nn;
        rc = propose_from_ctx(n, gen_parent, gen_age, &cx, seed, step, (uint32_t)i, pp, aa,
                              slot_t12 + 2 * i, slot_pair + i, slot_flag + i);
        if (rc != ORC_OK) goto done;
        slot_logL[i] = model == 0 ? orc_log_likelihood(n, L, codes, pp, aa, pi, u, NULL)
                                  : orc_log_likelihood_model(model, kappa, n, L, codes, pp, aa, pi, NULL);
        slot_S[i] = orc_coalescent_S(n, aa);
    }
    rc = orc_weights(N + 1, slot_logL, w, cum);
    if (rc != ORC_OK) goto done;
    for (d = 0; d < K; ++d) {
        double ud = orc_uniform(seed, 0u, step, ORC_TAG_DRAW, (uint32_t)d);
        draws[d] = orc_draw(N + 1, cum, ud, draw_flag + d);
        last = draws[d];
    }
    /* the last draw generates the next proposal set (Fig. 12) */
    memcpy(gen_parent, par_all + (size_t)last * nn, sizeof(int32_t) * (size_t)nn);
    memcpy(gen_age, age_all + (size_t)last * nn, sizeof(double) * (size_t)nn);
    *gen_logL = slot_logL[last];
done:
    ctx_free(&cx);
    free(par_all);
    free(age_all);
    free(w);
    free(cum);
    return rc;
}

int orc_gmh_step(int n, int L, const uint8_t* codes, const double pi[4], double u,
                 double theta0, int N, int K, uint64_t seed, uint32_t step,
                 int32_t* gen_parent, double* gen_age, double* gen_logL,
                 int32_t* out_target, double* slot_logL, double* slot_S, double* slot_t12,
                 int32_t* slot_pair, int32_t* slot_flag, int32_t* draws, int32_t* draw_flag) {
    return gmh_step_impl(0, 0.0, n, L, codes, pi, u, theta0, N, K, seed, step, gen_parent, gen_age,
                         gen_logL, out_target, slot_logL, slot_S, slot_t12, slot_pair, slot_flag,
                         draws, draw_flag);
}

/* The same step with P(D|G) under model 1 (F84) or 2 (HKY85): only the
   likelihood of Eq. 22 changes; proposals, weights and draws are those of Alg. 1. */
int orc_gmh_step_model(int model, double kappa, int n, int L, const uint8_t* codes,
                       const double pi[4], double theta0, int N, int K, uint64_t seed,
                       uint32_t step, int32_t* gen_parent, double* gen_age, double* gen_logL,
                       int32_t* out_target, double* slot_logL, double* slot_S, double* slot_t12,
                       int32_t* slot_pair, int32_t* slot_flag, int32_t* draws, int32_t* draw_flag) {
    if (model < 0 || model > 2) return ORC_E_ARG;
    return gmh_step_impl(model, kappa, n, L, codes, pi, orc_model_rate(model, kappa, pi), theta0, N,
                         K, seed, step, gen_parent, gen_age, gen_logL, out_target, slot_logL,
                         slot_S, slot_t12, slot_pair, slot_flag, draws, draw_flag);
}

/* Alg. 1 (L911-924) with Fig. 12's burn-in (L1312-1327; S17): burn-in steps draw once
   and store nothing, sampling steps draw min(N, remaining).  The generator
   gen_parent/gen_age is advanced in place.  n_flagged counts drawn items that were
   near a threshold; first_flag_step (nullable) receives the first step in which ANY
   slot choice or draw was flagged (-1 if none): up to that step the chain is
   determined by the algorithm, after it by the rounding of one comparison. */
int orc_run_chain(int n, int L, const uint8_t* codes, const double pi[4], double u,
                  double theta0, int N, int burnin, int M, uint64_t seed,
                  int32_t* gen_parent, double* gen_age, double* S_out, double* logL_out,
                  int64_t* step_out, int32_t* slot_out, int32_t* n_flagged,
                  int64_t* first_flag_step) {
    double gen_logL = orc_log_likelihood(n, L, codes, gen_parent, gen_age, pi, u, NULL);
    double* slot_logL = (double*)malloc(sizeof(double) * (size_t)(N + 1));
    double* slot_S = (double*)malloc(sizeof(double) * (size_t)(N + 1));
    double* slot_t12 = (double*)malloc(sizeof(double) * 2 * (size_t)(N + 1));
    int32_t* slot_pair = (int32_t*)malloc(sizeof(int32_t) * (size_t)(N + 1));
    int32_t* slot_flag = (int32_t*)malloc(sizeof(int32_t) * (size_t)(N + 1));
    int32_t* draws = (int32_t*)malloc(sizeof(int32_t) * (size_t)N);
    int32_t* dflag = (int32_t*)malloc(sizeof(int32_t) * (size_t)N);
    int stored = 0, rc = ORC_OK, d, target;
    uint32_t step = 0;
    *n_flagged = 0;
    if (first_flag_step) *first_flag_step = -1;
    while (stored < M || (int)step < burnin) {
        int burn = (int)step < burnin;
        int K = burn ? 1 : (M - stored < N ? M - stored : N);
        rc = orc_gmh_step(n, L, codes, pi, u, theta0, N, K, seed, step, gen_parent, gen_age,
                          &gen_logL, &target, slot_logL, slot_S, slot_t12, slot_pair, slot_flag,
                          draws, dflag);
        if (rc != ORC_OK) break;
        if (first_flag_step && *first_flag_step < 0) {
            for (d = 0; d < K; ++d)
                if (dflag[d]) *first_flag_step = step;
            for (d = 1; d <= N; ++d)
                if (slot_flag[d]) *first_flag_step = step;
        }
        for (d = 0; d < K; ++d) {
            if (dflag[d] || slot_flag[draws[d]]) (*n_flagged)++;
            if (burn) continue;
            S_out[stored] = slot_S[draws[d]];
            logL_out[stored] = slot_logL[draws[d]];
            step_out[stored] = step;
            slot_out[stored] = draws[d];
            stored++;
        }
        step++;
    }
    free(slot_logL);
    free(slot_S);
    free(slot_t12);
    free(slot_pair);
    free(slot_flag);
    free(draws);
    free(dflag);
    return rc;
}

/* ------------------------------------------------------------------------- */
/* Relative likelihood and its maximum (2.5 L752-797, 5.1.5, 5.2.3; S20).      */
/* ------------------------------------------------------------------------- */

/* Eq. 25-26: ln L(theta) = ln( (1/M) sum_G P(G|theta)/P(G|theta0) ), with Eq. 18. */
double orc_log_rel_likelihood(int M, const double* S, int n, double theta0, double theta) {
    double* terms = (double*)malloc(sizeof(double) * (size_t)M);
    double r;
    int g;
    for (g = 0; g < M; ++g)
        terms[g] = (double)(n - 1) * log(theta0 / theta) - S[g] * (1.0 / theta - 1.0 / theta0);
    r = log_sum_exp(terms, M) - log((double)M);
    free(terms);
    return r;
}

/* sum_G w_G S_G / sum_G w_G with w_G proportional to P(G|theta)/P(G|theta0) */
double orc_weighted_mean_S(int M, const double* S, double theta0, double theta) {
    double mx = -INFINITY, num = 0.0, den = 0.0;
    int g;
    for (g = 0; g < M; ++g) {
        double e = -S[g] * (1.0 / theta - 1.0 / theta0);
        if (e > mx) mx = e;
    }
    for (g = 0; g < M; ++g) {
        double w = exp(-S[g] * (1.0 / theta - 1.0 / theta0) - mx);
        num += w * S[g];
        den += w;
    }
    return num / den;
}

/* EM fixed-point map theta <- S_w(theta)/(n-1) (stationarity of ln L) */
double orc_em_map(int M, const double* S, int n, double theta0, double theta) {
    return orc_weighted_mean_S(M, S, theta0, theta) / (double)(n - 1);
}

/* d ln L / d theta has the sign of S_w(theta) - (n-1) theta */
static double stationarity(int M, const double* S, int n, double theta0, double theta) {
    return orc_weighted_mean_S(M, S, theta0, theta) - (double)(n - 1) * theta;
}

double orc_theta_hat(int M, const double* S, int n, double theta0, int G,
                     double* grid_theta, double* grid_ll) {
    double smin = INFINITY, smax = -INFINITY, lo, hi, best_ll = -INFINITY;
    int g, best = 0, it;
    for (g = 0; g < M; ++g) {
        if (S[g] < smin) smin = S[g];
        if (S[g] > smax) smax = S[g];
    }
    if (smin == smax || G < 3) return smin / (double)(n - 1);
    /* every stationary point lies in [S_min, S_max]/(n-1) (Appendix B) */
    for (g = 0; g < G; ++g) {
        double th = exp(log(smin / (n - 1)) + (log(smax / (n - 1)) - log(smin / (n - 1))) * g / (G - 1));
        double ll = orc_log_rel_likelihood(M, S, n, theta0, th);
        if (grid_theta) grid_theta[g] = th;
        if (grid_ll) grid_ll[g] = ll;
        if (ll > best_ll) {
            best_ll = ll;
            best = g;
        }
    }
    lo = exp(log(smin / (n - 1)) + (log(smax / (n - 1)) - log(smin / (n - 1))) * (best > 0 ? best - 1 : 0) / (G - 1));
    hi = exp(log(smin / (n - 1)) + (log(smax / (n - 1)) - log(smin / (n - 1))) * (best < G - 1 ? best + 1 : G - 1) / (G - 1));
    if (best == 0) lo = smin / (n - 1);
    if (best == G - 1) hi = smax / (n - 1);
    if (stationarity(M, S, n, theta0, lo) >= 0.0 && stationarity(M, S, n, theta0, hi) <= 0.0) {
        /* bisection on the sign of the derivative */
        for (it = 0; it < 200 && hi - lo > 1e-15 * hi; ++it) {
            double mid = 0.5 * (lo + hi);
            if (stationarity(M, S, n, theta0, mid) >= 0.0) lo = mid;
            else hi = mid;
        }
        return 0.5 * (lo + hi);
    }
    /* golden-section search on ln L inside the bracket */
    {
        const double gr = 0.6180339887498949;
        double a = lo, b = hi, c = b - gr * (b - a), d = a + gr * (b - a);
        for (it = 0; it < 300 && b - a > 1e-15 * b; ++it) {
            if (orc_log_rel_likelihood(M, S, n, theta0, c) > orc_log_rel_likelihood(M, S, n, theta0, d)) b = d;
            else a = c;
            c = b - gr * (b - a);
            d = a + gr * (b - a);
        }
        return 0.5 * (a + b);
    }
}

/*
 * EM re-drive of Fig. 11 (L1208-1225) and L791-797: n_iter times
 * { sample with the driving value theta (Alg. 1 + burn-in, seed + it); theta-hat =
 * argmax of Eq. 25 over those samples; theta0 <- theta-hat }.  The genealogy carries
 * over between iterations (gen_parent / gen_age advanced in place); every iteration
 * restarts its step counter at 0 with its own seed.  theta_trace[it] = that
 * iteration's estimate; first_flag[it] = orc_run_chain's first flagged step (-1 none).
 * S_buf: caller scratch of M doubles.
 */
int orc_em(int n, int L, const uint8_t* codes, const double pi[4], double u, double theta0,
           int N, int burnin, int M, uint64_t seed, int n_iter, int G, int32_t* gen_parent,
           double* gen_age, double* theta_trace, int64_t* first_flag) {
    double* S = (double*)malloc(sizeof(double) * (size_t)M);
    double* lL = (double*)malloc(sizeof(double) * (size_t)M);
    int64_t* st = (int64_t*)malloc(sizeof(int64_t) * (size_t)M);
    int32_t* sl = (int32_t*)malloc(sizeof(int32_t) * (size_t)M);
    double theta = theta0;
    int it, rc = ORC_OK;
    int32_t nf;
    for (it = 0; it < n_iter; ++it) {
        rc = orc_run_chain(n, L, codes, pi, u, theta, N, burnin, M, seed + (uint64_t)it, gen_parent,
                           gen_age, S, lL, st, sl, &nf, first_flag + it);
        if (rc != ORC_OK) break;
        theta = orc_theta_hat(M, S, n, theta, G, NULL, NULL);
        theta_trace[it] = theta;
    }
    free(S);
    free(lL);
    free(st);
    free(sl);
    return rc;
}

/*
 * Multiple loci: loci with independent genealogies share theta, so
 * the joint relative likelihood is the product over loci of Eq. 25 (L765-797), each
 * locus l with its own samples S_l[0..M_l), n_l and driving value theta0_l.  The
 * samples are concatenated: locus l starts at sum_{k<l} M_k.
 */
double orc_log_rel_likelihood_loci(int K, const int* M, const double* S, const int* n,
                                   const double* theta0, double theta) {
    double r = 0.0;
    int l;
    long off = 0;
    for (l = 0; l < K; ++l) {
        r += orc_log_rel_likelihood(M[l], S + off, n[l], theta0[l], theta);
        off += M[l];
    }
    return r;
}

/* d ln L / d theta = sum_l (S_w,l(theta) - (n_l - 1) theta) / theta^2: the sign of the sum */
static double stationarity_loci(int K, const int* M, const double* S, const int* n,
                                const double* theta0, double theta) {
    double f = 0.0;
    int l;
    long off = 0;
    for (l = 0; l < K; ++l) {
        f += stationarity(M[l], S + off, n[l], theta0[l], theta);
        off += M[l];
    }
    return f;
}

/* Joint theta-hat: global argmax over [sum_l S_min,l, sum_l S_max,l] / sum_l (n_l - 1)
   (every stationary point solves sum_l S_w,l = theta sum_l (n_l - 1)), by the same
   grid + bisection (else golden section) as orc_theta_hat. */
double orc_theta_hat_loci(int K, const int* M, const double* S, const int* n,
                          const double* theta0, int G, double* grid_theta, double* grid_ll) {
    double smin = 0.0, smax = 0.0, dof = 0.0, lo, hi, best_ll = -INFINITY, a0, a1;
    int g, l, best = 0, it;
    long off = 0;
    for (l = 0; l < K; ++l) {
        double mn = INFINITY, mx = -INFINITY;
        for (g = 0; g < M[l]; ++g) {
            if (S[off + g] < mn) mn = S[off + g];
            if (S[off + g] > mx) mx = S[off + g];
        }
        smin += mn;
        smax += mx;
        dof += (double)(n[l] - 1);
        off += M[l];
    }
    a0 = smin / dof;
    a1 = smax / dof;
    if (a0 == a1 || G < 3) return a0;
    for (g = 0; g < G; ++g) {
        double th = exp(log(a0) + (log(a1) - log(a0)) * g / (G - 1));
        double ll = orc_log_rel_likelihood_loci(K, M, S, n, theta0, th);
        if (grid_theta) grid_theta[g] = th;
        if (grid_ll) grid_ll[g] = ll;
        if (ll > best_ll) {
            best_ll = ll;
            best = g;
        }
    }
    lo = best > 0 ? exp(log(a0) + (log(a1) - log(a0)) * (best - 1) / (G - 1)) : a0;
    hi = best < G - 1 ? exp(log(a0) + (log(a1) - log(a0)) * (best + 1) / (G - 1)) : a1;
    if (stationarity_loci(K, M, S, n, theta0, lo) >= 0.0 &&
        stationarity_loci(K, M, S, n, theta0, hi) <= 0.0) {
        for (it = 0; it < 200 && hi - lo > 1e-15 * hi; ++it) {
            double mid = 0.5 * (lo + hi);
            if (stationarity_loci(K, M, S, n, theta0, mid) >= 0.0) lo = mid;
            else hi = mid;
        }
        return 0.5 * (lo + hi);
    }
    {
        const double gr = 0.6180339887498949;
        double a = lo, b = hi, c = b - gr * (b - a), d = a + gr * (b - a);
        for (it = 0; it < 300 && b - a > 1e-15 * b; ++it) {
            if (orc_log_rel_likelihood_loci(K, M, S, n, theta0, c) >
                orc_log_rel_likelihood_loci(K, M, S, n, theta0, d)) b = d;
            else a = c;
            c = b - gr * (b - a);
            d = a + gr * (b - a);
        }
        return 0.5 * (a + b);
    }
}

/*
 * Algorithm 2 (L1329-1340) literally, on ln L, with delta = 1e-6 theta0 and
 * eps = 1e-9 theta0 (S20).  A cross-check only: a local ascent from theta0.
 */
double orc_theta_alg2(int M, const double* S, int n, double theta0, int max_iter) {
    double delta = 1e-6 * theta0, eps = 1e-9 * theta0;
    double theta, theta_next = theta0, grad;
    int it = 0, inner;
    do {
        theta = theta_next;
        grad = (orc_log_rel_likelihood(M, S, n, theta0, theta_next + delta) -
                orc_log_rel_likelihood(M, S, n, theta0, theta_next - delta)) / (2.0 * delta);
        inner = 0;
        while ((orc_log_rel_likelihood(M, S, n, theta0, theta_next) -
                    orc_log_rel_likelihood(M, S, n, theta0, theta_next + grad) > delta ||
                theta_next + grad < 0.0) && inner < 200) {
            grad = grad / 2.0;
            inner++;
        }
        theta_next = theta_next + grad;
        it++;
    } while (fabs(theta - theta_next) > eps && it < max_iter);
    return theta_next;
}

/* ------------------------------------------------------------------------- */
/* UPGMA (5.1.3 L1287-1295; S19): Hamming distances, average linkage,         */
/* height = theta0 * D / 2, forced strictly above the children.               */
/* ------------------------------------------------------------------------- */
int orc_upgma(int n, int L, const uint8_t* codes, double theta0, int32_t* parent, double* age) {
    int nn = 2 * n - 1, i, j, s, step;
    double* D = (double*)malloc(sizeof(double) * (size_t)nn * (size_t)nn);
    int* size = (int*)calloc((size_t)nn, sizeof(int));
    int* alive = (int*)calloc((size_t)nn, sizeof(int));
    if (n < 2) {
        free(D);
        free(size);
        free(alive);
        return ORC_E_ARG;
    }
    for (i = 0; i < nn; ++i) {
        parent[i] = -1;
        age[i] = 0.0;
    }
    for (i = 0; i < n; ++i) {
        size[i] = 1;
        alive[i] = 1;
        for (j = 0; j < n; ++j) {
            int diff = 0;
            for (s = 0; s < L; ++s) {   /* a difference: disjoint base sets (S24) */
                int a = codes[(long)i * L + s], b = codes[(long)j * L + s];
                int sa = a < 4 ? 1 << a : a - 16, sb = b < 4 ? 1 << b : b - 16;
                diff += (sa & sb) == 0;
            }
            D[i * nn + j] = (double)diff;
        }
    }
    for (step = 0; step < n - 1; ++step) {
        int bi = -1, bj = -1, v = n + step;
        double best = INFINITY, h;
        for (i = 0; i < v; ++i) {
            if (!alive[i]) continue;
            for (j = i + 1; j < v; ++j) {
                if (!alive[j]) continue;
                if (D[i * nn + j] < best) {   /* strict: ties keep the smallest (i, j) */
                    best = D[i * nn + j];
                    bi = i;
                    bj = j;
                }
            }
        }
        h = theta0 * best / 2.0;
        if (h < age[bi] + 1e-6 * theta0) h = age[bi] + 1e-6 * theta0;
        if (h < age[bj] + 1e-6 * theta0) h = age[bj] + 1e-6 * theta0;
        age[v] = h;
        parent[bi] = v;
        parent[bj] = v;
        alive[bi] = alive[bj] = 0;
        alive[v] = 1;
        size[v] = size[bi] + size[bj];
        for (i = 0; i < v; ++i) {
            double d;
            if (!alive[i]) continue;
            /* mean over all leaf pairs across the two clusters (L1290-1292) */
            d = (size[bi] * D[bi * nn + i] + size[bj] * D[bj * nn + i]) / (double)size[v];
            D[v * nn + i] = d;
            D[i * nn + v] = d;
        }
    }
    free(D);
    free(size);
    free(alive);
    return ORC_OK;
}

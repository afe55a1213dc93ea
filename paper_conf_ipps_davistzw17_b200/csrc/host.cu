// host.cu -- the C ABI (include/mpcgs.h): validation, model setup, G0, device
// workspace layout, the device-resident step loop, theta estimation, NCCL.
//
// Host code here never computes the method's hot path: every per-step
// quantity (targets, contexts, proposals, likelihoods, weights, draws, theta
// curve) is computed by the kernels in step.cu / prune.cu / theta.cu.  The host
// builds G0 (UPGMA, 5.1.3 L1287-1295) and the post-order schedule of trees it
// is handed (mpcgs_score_trees / set_state), and drives Newton on the theta
// bracket with device reductions.
#include <dlfcn.h>
#include <nccl.h>
#include <nvtx3/nvToolsExt.h>  // header-only NVTX v3: ranges show in nsys / ncu --nvtx

#include <algorithm>
#include <chrono>
#include <thread>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <string>
#include <vector>

#include "common.cuh"
#include "kernels.cuh"
#include "mpcgs.h"

using namespace mpcgs;

// ---------------------------------------------------------------- NCCL (dlopen)
namespace {
struct NcclApi {
    bool ok = false;
    ncclResult_t (*getUniqueId)(ncclUniqueId*) = nullptr;
    ncclResult_t (*commInitRank)(ncclComm_t*, int, ncclUniqueId, int) = nullptr;
    ncclResult_t (*allGather)(const void*, void*, size_t, ncclDataType_t, ncclComm_t, cudaStream_t) = nullptr;
    ncclResult_t (*commDestroy)(ncclComm_t) = nullptr;
    const char* (*errStr)(ncclResult_t) = nullptr;
};
NcclApi& nccl() {
    static NcclApi api;
    static bool tried = false;
    if (!tried) {
        tried = true;
        void* h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_GLOBAL);
        if (!h) h = dlopen("libnccl.so", RTLD_NOW | RTLD_GLOBAL);
        if (h) {
            api.getUniqueId = (decltype(api.getUniqueId))dlsym(h, "ncclGetUniqueId");
            api.commInitRank = (decltype(api.commInitRank))dlsym(h, "ncclCommInitRank");
            api.allGather = (decltype(api.allGather))dlsym(h, "ncclAllGather");
            api.commDestroy = (decltype(api.commDestroy))dlsym(h, "ncclCommDestroy");
            api.errStr = (decltype(api.errStr))dlsym(h, "ncclGetErrorString");
            api.ok = api.getUniqueId && api.commInitRank && api.allGather && api.commDestroy;
        }
    }
    return api;
}
}  // namespace

// ---------------------------------------------------------------- context
struct mpcgs_ctx {
    DevState s{};
    int n = 0, L = 0, nn = 0, Lpad = 0, nops = 0, depth = 0, precision = 64;
    int world = 1, rank = 0, burnin = 0;
    bool incremental = false;
    int model = 0;           // MPCGS_MODEL_*
    double kappa = 0.0;
    int L_orig = 0;          // alignment columns (L = scored sites: patterns if compressed)
    int Nmax = 0;
    int64_t Mmax = 0;
    double theta0 = 0.0, sample_theta0 = 0.0;
    cudaStream_t user = nullptr, work = nullptr;
    void* ws = nullptr;
    size_t ws_bytes = 0;
    bool own_ws = false;
    double* score_out = nullptr;
    unsigned* theta_cnt = nullptr;
    uint32_t* codes2 = nullptr;
    int64_t nsamples = 0;
    int lastN = 0;
    bool sticky = false;
    std::string err;
    ncclComm_t comm = nullptr;
    int timing = 0;              // bit 0: events per step / prune launch; bit 1: flush L2 between steps
    void* flush_buf = nullptr;   // 256 MiB scratch written between timed steps (> 126 MB L2)
    double loop_ms = 0.0, prune_ms = 0.0, propose_ms = 0.0, draw_ms = 0.0;
    int graph_steps = 32;
    int64_t launches = 0;
    std::vector<cudaEvent_t> evpool;
    cudaEvent_t ev_a = nullptr, ev_b = nullptr;
    std::vector<double> pinned_dummy;
    // a sampling loop enqueued by sample_begin and not yet finished by sample_end
    struct {
        bool active = false;
        cudaGraph_t graph = nullptr;
        cudaGraphExec_t exec = nullptr;
        cudaEvent_t end = nullptr;
        int N = 0;
        int64_t M = 0;
        int64_t stored = 0;  // samples in the store once the loop's last step is done
    } pend;
};

namespace {

// NVTX range for the duration of an entry point (tracing)
struct NvtxRange {
    explicit NvtxRange(const char* name) { nvtxRangePushA(name); }
    ~NvtxRange() { nvtxRangePop(); }
};

mpcgs_status fail(mpcgs_ctx* c, mpcgs_status st, const std::string& msg) {
    if (c) {
        c->err = msg;
        if (st == MPCGS_E_CUDA || st == MPCGS_E_NCCL) c->sticky = true;
    }
    return st;
}

#define CU(call)                                                                                  \
    do {                                                                                          \
        cudaError_t e_ = (call);                                                                  \
        if (e_ != cudaSuccess)                                                                    \
            return fail(c, MPCGS_E_CUDA, std::string(#call) + ": " + cudaGetErrorString(e_));      \
    } while (0)

#define CHECK_CTX(c)                                                               \
    do {                                                                           \
        if (!(c)) return MPCGS_E_ARG;                                              \
        if ((c)->sticky) return MPCGS_E_CUDA;                                      \
    } while (0)

// ------------------------------------------------------------ workspace layout
struct Layout {
    size_t codes, codes2, parent, left, right, need, age, e, em, gen, ctx_i, ctx_d, tau, len, lcnt, entry, omega, fixed;
    size_t gm, sched_P;
    size_t tree_need, rec, sched_op, sched_e, tree_acc, tile_cnt, sS, sL, sStep, sSlot, counters, last_draws, theta_buf,
        theta_cnt, score_out, site_w, GL, GE, path, pathsib, cpath, csib, ixyz, iee, cinfo, gen_order, total;
    int tiles_max;
};

size_t al(size_t x) { return (x + 255) & ~(size_t)255; }

// 2-bit packed tip codes, 16 sites per 32-bit word, rows padded past the last tile
int codes2_words(int L) { return ((L + 4096 + 63) / 64) * 4; }

Layout layout(int n, int L, int Nmax, int64_t Mmax, int precision, int incremental = 0, int model = 0) {
    Layout y{};
    const int nn = 2 * n - 1, nops = n - 1;
    const int Lpad = (L + 15) & ~15;
    const size_t esz = precision == 32 ? sizeof(float4) : sizeof(double4);
    y.tiles_max = (L + PRUNE_THREADS - 1) / PRUNE_THREADS;
    size_t o = 0;
    auto take = [&](size_t bytes) {
        size_t r = o;
        o += al(bytes);
        return r;
    };
    y.codes = take((size_t)n * Lpad);
    y.codes2 = take(8 * (size_t)n * codes2_words(L));  // room for 4-bit base-set codes (ambiguity data)
    y.parent = take(4 * (size_t)nn);
    y.left = take(4 * (size_t)nn);
    y.right = take(4 * (size_t)nn);
    y.need = take(4 * (size_t)nn);
    y.age = take(8 * (size_t)nn);
    y.e = take(8 * (size_t)nn);
    y.em = take(8 * (size_t)nn);
    y.gen = take(8 * 4);
    y.ctx_i = take(4 * 16);
    y.ctx_d = take(8 * 8);
    y.tau = take(8 * (size_t)(n + 2));
    y.len = take(8 * (size_t)(n + 1));
    y.lcnt = take(4 * (size_t)(n + 1));
    y.entry = take(4 * (size_t)(n + 2));
    y.omega = take(8 * 16 * (size_t)(n + 1));  // OM_STRIDE doubles per interval (step_body.cuh)
    y.fixed = take(8 * (size_t)n);
    y.rec = take(8 * REC * (size_t)(Nmax + 1));
    y.tree_need = take(4 * (size_t)Nmax);
    y.sched_op = take(4 * (size_t)Nmax * nops);
    y.sched_e = take(esz * (size_t)Nmax * nops);
    y.tree_acc = take(32 * (size_t)Nmax);
    y.tile_cnt = take(4 * (size_t)Nmax);
    y.sS = take(8 * (size_t)std::max<int64_t>(Mmax, 1));
    y.sL = take(8 * (size_t)std::max<int64_t>(Mmax, 1));
    y.sStep = take(8 * (size_t)std::max<int64_t>(Mmax, 1));
    y.sSlot = take(4 * (size_t)std::max<int64_t>(Mmax, 1));
    y.counters = take(8 * 8);
    y.last_draws = take(4 * (size_t)Nmax);
    y.theta_buf = take(8 * (size_t)(2 * MPCGS_MAX_GRID + 3 * 296 + 16));
    y.theta_cnt = take(16);
    y.score_out = take(8 * (size_t)Nmax);
    y.site_w = take(8 * (size_t)L);
    const size_t tsz = precision == 32 ? 4 : 8;
    y.GL = take(incremental ? 4 * tsz * (size_t)(n - 1) * Lpad : 0);
    y.GE = take(incremental ? 4 * (size_t)(n - 1) * Lpad : 0);
    y.path = take(4 * (size_t)n);
    y.pathsib = take(4 * (size_t)n);
    y.cpath = take(4 * (size_t)n);
    y.csib = take(4 * (size_t)n);
    y.ixyz = take(16 * (size_t)Nmax);
    y.iee = take(80 * (size_t)Nmax);
    y.cinfo = take(32);
    y.gen_order = take(4 * (size_t)n);
    y.gm = take(model ? 8 * 48 : 0);
    y.sched_P = take(model ? 16 * tsz * 2 * (size_t)Nmax * nops : 0);
    y.total = o;
    return y;
}

// ------------------------------------------------------------ substitution models (f4)
// Rate matrix of the model (i != j; rows sum to 0), scaled to one expected
// substitution per unit time (S3).  Purines A, G = 0, 2; pyrimidines C, T = 1, 3.
//   F84   (Felsenstein 1984): q_ij = pi_j (1 + kappa / Pi_{g(j)} [g(i) = g(j)])
//   HKY85 (Hasegawa, Kishino & Yano 1985): q_ij = pi_j (kappa [g(i) = g(j)] + [g(i) != g(j)])
void rate_matrix(int model, double kappa, const double pi[4], double Q[16]) {
    auto grp = [](int x) { return x & 1; };
    const double Pi[2] = {pi[0] + pi[2], pi[1] + pi[3]};
    double flux = 0.0;
    for (int i = 0; i < 4; ++i) {
        double row = 0.0;
        for (int j = 0; j < 4; ++j) {
            if (i == j) continue;
            const bool ts = grp(i) == grp(j);
            double q;
            if (model == MPCGS_MODEL_F84) q = pi[j] * (1.0 + (ts ? kappa / Pi[grp(j)] : 0.0));
            else if (model == MPCGS_MODEL_HKY85) q = pi[j] * (ts ? kappa : 1.0);
            else q = pi[j];  // F81
            Q[i * 4 + j] = q;
            row += q;
        }
        Q[i * 4 + i] = -row;
        flux += pi[i] * row;
    }
    const double scale = flux > 0.0 ? 1.0 / flux : 1.0;
    for (int k = 0; k < 16; ++k) Q[k] *= scale;
}

// Structured constants of F84 / HKY85 (gm[36..40], read by the table kernel): with
// the rate matrix normalised by s (rate_matrix), P(t) v has the closed form
//   (P(t) v)_i = (1 - e^{-s t}) T + (e^{-s t} - e^{-s A_g t}) G_g / Pi_g + e^{-s A_g t} v_i,
// T = pi . v, G_g = sum_{j in g} pi_j v_j, g = the purine / pyrimidine group of i:
// Q = s [J + kappa K - (1 + kappa) I] for F84 (J = 1 pi^T, K_ij = [same group] pi_j / Pi_g,
// commuting projections with JK = KJ = J) gives A_R = A_Y = 1 + kappa; HKY85 gives
// A_g = 1 + Pi_g (kappa - 1) (Hasegawa, Kishino & Yano 1985).  {s, A_R, A_Y, Pi_R, Pi_Y}.
void model_consts(int model, double kappa, const double pi[4], double out[5]) {
    double Q[16];
    rate_matrix(model, kappa, pi, Q);
    // rate_matrix scales the unnormalised rates by s: recover s from one off-diagonal entry
    // (q_01 = s pi_1, a transversion in both models)
    const double s = Q[0 * 4 + 1] / pi[1];
    const double PiR = pi[0] + pi[2], PiY = pi[1] + pi[3];
    out[0] = s;
    out[1] = model == MPCGS_MODEL_F84 ? 1.0 + kappa : 1.0 + PiR * (kappa - 1.0);
    out[2] = model == MPCGS_MODEL_F84 ? 1.0 + kappa : 1.0 + PiY * (kappa - 1.0);
    out[3] = PiR;
    out[4] = PiY;
}

// Eigen-system of a reversible Q: S = D^1/2 Q D^-1/2 (D = diag pi) is symmetric;
// cyclic Jacobi gives S = U diag(ev) U^T, so P(t) = e^{Qt} = V diag(e^{ev t}) W with
// V = D^-1/2 U and W = U^T D^1/2.  gm = {ev[4], V[16], W[16]}.  Needs pi > 0.
void eigen_system(const double Q[16], const double pi[4], double gm[36]) {
    double A[16], U[16];
    for (int i = 0; i < 4; ++i)
        for (int j = 0; j < 4; ++j) {
            A[i * 4 + j] = std::sqrt(pi[i] / pi[j]) * Q[i * 4 + j];
            U[i * 4 + j] = i == j ? 1.0 : 0.0;
        }
    for (int i = 0; i < 4; ++i)  // exact symmetry (rounding)
        for (int j = i + 1; j < 4; ++j) A[i * 4 + j] = A[j * 4 + i] = 0.5 * (A[i * 4 + j] + A[j * 4 + i]);
    for (int sweep = 0; sweep < 64; ++sweep) {
        double off = 0.0;
        for (int i = 0; i < 4; ++i)
            for (int j = i + 1; j < 4; ++j) off += A[i * 4 + j] * A[i * 4 + j];
        if (off < 1e-300) break;
        for (int p = 0; p < 4; ++p)
            for (int q = p + 1; q < 4; ++q) {
                const double apq = A[p * 4 + q];
                if (apq == 0.0) continue;
                const double th = (A[q * 4 + q] - A[p * 4 + p]) / (2.0 * apq);
                const double t = (th >= 0.0 ? 1.0 : -1.0) / (std::fabs(th) + std::sqrt(th * th + 1.0));
                const double cs = 1.0 / std::sqrt(t * t + 1.0), sn = t * cs;
                for (int k = 0; k < 4; ++k) {  // A <- J^T A J (columns, then rows)
                    const double akp = A[k * 4 + p], akq = A[k * 4 + q];
                    A[k * 4 + p] = cs * akp - sn * akq;
                    A[k * 4 + q] = sn * akp + cs * akq;
                }
                for (int k = 0; k < 4; ++k) {
                    const double apk = A[p * 4 + k], aqk = A[q * 4 + k];
                    A[p * 4 + k] = cs * apk - sn * aqk;
                    A[q * 4 + k] = sn * apk + cs * aqk;
                }
                for (int k = 0; k < 4; ++k) {  // U <- U J
                    const double ukp = U[k * 4 + p], ukq = U[k * 4 + q];
                    U[k * 4 + p] = cs * ukp - sn * ukq;
                    U[k * 4 + q] = sn * ukp + cs * ukq;
                }
            }
    }
    for (int k = 0; k < 4; ++k) gm[k] = std::min(A[k * 4 + k], 0.0);  // Q is negative semi-definite
    for (int i = 0; i < 4; ++i)
        for (int k = 0; k < 4; ++k) {
            gm[4 + i * 4 + k] = U[i * 4 + k] / std::sqrt(pi[i]);
            gm[20 + k * 4 + i] = U[i * 4 + k] * std::sqrt(pi[i]);
        }
}

// ------------------------------------------------------------ host tree helpers
int check_tree(int n, const int32_t* parent, const double* age, std::string& why) {
    const int nn = 2 * n - 1;
    std::vector<int> kids(nn, 0);
    int roots = 0;
    for (int v = 0; v < nn; ++v) {
        const int p = parent[v];
        if (p < 0) {
            ++roots;
            if (v < n) { why = "a tip has no parent"; return -1; }
            continue;
        }
        if (p < n || p >= nn) { why = "parent id out of the interior range"; return -1; }
        if (!(age[p] >= age[v])) { why = "a parent is younger than its child"; return -1; }
        if (!std::isfinite(age[v])) { why = "non-finite age"; return -1; }
        ++kids[p];
    }
    if (roots != 1) { why = "tree must have exactly one root"; return -1; }
    for (int v = 0; v < n; ++v)
        if (age[v] != 0.0) { why = "tips must have age 0 (S22)"; return -1; }
    for (int v = n; v < nn; ++v)
        if (kids[v] != 2) { why = "interior nodes need two children"; return -1; }
    // acyclic: every node reaches the root in < nn steps
    for (int v = 0; v < nn; ++v) {
        int x = v, k = 0;
        while (parent[x] >= 0 && k < nn) { x = parent[x]; ++k; }
        if (k >= nn) { why = "cycle in parent array"; return -1; }
    }
    return 0;
}

// Newick G0 (SURVEY 8(b) init_newick; the paper reads its initial genealogy from
// UPGMA, 5.1.3 L1287-1295, and its test data come with ms's Newick trees, L1499).
// Grammar: tree := node [':' len] ';'   node := '(' node ',' node ')' [label] | label,
// each non-root node with ':' length >= 0.  Tip labels are row indices "0".."n-1".
// Tips are contemporaneous (S22): every tip depth must agree with the deepest to
// 1e-5 of the height; a node's age is the longest path from it down to a tip, so
// ages never decrease towards the root.  Interior ids n..2n-2 ascend with age (ties:
// post-order), the creation order of a coalescent simulation.  0 or -1 with `why`.
int parse_newick(int n, const char* text, int32_t* parent, double* age, std::string& why) {
    struct Nd { int par = -1, c0 = -1, c1 = -1, tip = -1; double len = 0.0; };
    std::vector<Nd> nd;
    nd.reserve(2 * (size_t)n);
    const char* p = text;
    auto ws = [&]() { while (*p == ' ' || *p == '\t' || *p == '\n' || *p == '\r') ++p; };
    auto label = [&](std::string& out) {
        out.clear();
        while (*p && !std::strchr("(),:; \t\r\n", *p)) out.push_back(*p++);
    };
    auto number = [&](double& v) -> bool {
        char* end = nullptr;
        v = std::strtod(p, &end);
        if (end == p) return false;
        p = end;
        return std::isfinite(v) && v >= 0.0;
    };
    std::vector<char> seen(n, 0);
    std::vector<int> stack;  // open internal nodes
    int root = -1;
    std::string lab;
    // iterative parse: each node is created when first reached
    auto new_node = [&](int par) {
        nd.push_back(Nd{});
        const int id = (int)nd.size() - 1;
        nd[id].par = par;
        if (par >= 0) {
            if (nd[par].c0 < 0) nd[par].c0 = id;
            else if (nd[par].c1 < 0) nd[par].c1 = id;
            else return -2;  // multifurcation
        }
        return id;
    };
    auto parse_len = [&](int id) -> bool {
        ws();
        if (*p == ':') {
            ++p;
            ws();
            if (!number(nd[id].len)) return false;
        } else if (nd[id].par >= 0) {
            return false;  // every branch needs a length
        }
        return true;
    };
    ws();
    int cur_par = -1;
    for (;;) {
        ws();
        if ((int)nd.size() > 2 * n) { why = "more nodes than 2n-1"; return -1; }
        if (*p == '(') {
            ++p;
            const int id = new_node(cur_par);
            if (id == -2) { why = "a node has more than two children"; return -1; }
            if (cur_par < 0) root = id;
            stack.push_back(id);
            cur_par = id;
            continue;
        }
        // a tip
        label(lab);
        if (lab.empty()) { why = std::string("expected a tip label at '") + std::string(p, std::min<size_t>(16, std::strlen(p))) + "'"; return -1; }
        char* end = nullptr;
        const long t = std::strtol(lab.c_str(), &end, 10);
        if (*end || t < 0 || t >= n) { why = "tip label '" + lab + "' is not a row index 0..n-1"; return -1; }
        if (seen[t]) { why = "tip " + lab + " appears twice"; return -1; }
        seen[t] = 1;
        const int id = new_node(cur_par);
        if (id == -2) { why = "a node has more than two children"; return -1; }
        if (cur_par < 0) { why = "the tree is a single tip"; return -1; }
        nd[id].tip = (int)t;
        if (!parse_len(id)) { why = "tip " + lab + ": missing or invalid branch length"; return -1; }
        // close groups
        for (;;) {
            ws();
            if (*p == ',') {
                ++p;
                break;  // next sibling under cur_par
            }
            if (*p == ')') {
                ++p;
                const int done = stack.back();
                stack.pop_back();
                if (nd[done].c1 < 0) { why = "an internal node has one child"; return -1; }
                label(lab);  // optional internal label, ignored
                if (!parse_len(done)) { why = "internal node: missing or invalid branch length"; return -1; }
                cur_par = stack.empty() ? -1 : stack.back();
                if (stack.empty()) break;
                continue;
            }
            if (*p == ';' && stack.empty()) break;
            why = std::string("unexpected character '") + (*p ? *p : '0') + "'";
            return -1;
        }
        if (stack.empty()) break;
    }
    ws();
    if (*p != ';') { why = "missing ';'"; return -1; }
    if ((int)nd.size() != 2 * n - 1) { why = "the tree must have n tips and n-1 binary internal nodes"; return -1; }
    for (int t = 0; t < n; ++t)
        if (!seen[t]) { why = "tip " + std::to_string(t) + " missing"; return -1; }
    const int m = (int)nd.size();
    std::vector<double> depth(m, 0.0), h(m, 0.0);
    for (int v = 0; v < m; ++v)  // parents precede children in creation order
        if (nd[v].par >= 0) depth[v] = depth[nd[v].par] + nd[v].len;
    double height = 0.0;
    for (int v = 0; v < m; ++v)
        if (nd[v].tip >= 0) height = std::max(height, depth[v]);
    for (int v = 0; v < m; ++v)
        if (nd[v].tip >= 0 && height - depth[v] > 1e-5 * height) { why = "tips are not contemporaneous (S22)"; return -1; }
    // age = longest path down to a tip; children are created after their parent
    std::vector<int> post;  // post-order (children before parents)
    {
        std::vector<std::pair<int, int>> st{{root, 0}};
        while (!st.empty()) {
            auto& [v, k] = st.back();
            if (nd[v].tip < 0 && k < 2) {
                const int ch = k == 0 ? nd[v].c0 : nd[v].c1;
                ++k;
                st.push_back({ch, 0});
                continue;
            }
            post.push_back(v);
            st.pop_back();
        }
    }
    std::vector<int> interior;
    for (int v : post) {
        if (nd[v].tip >= 0) continue;
        h[v] = std::max(h[nd[v].c0] + nd[nd[v].c0].len, h[nd[v].c1] + nd[nd[v].c1].len);
        interior.push_back(v);
    }
    std::stable_sort(interior.begin(), interior.end(), [&](int a, int b) { return h[a] < h[b]; });
    std::vector<int> id(m, -1);
    for (int v = 0; v < m; ++v)
        if (nd[v].tip >= 0) id[v] = nd[v].tip;
    for (size_t k = 0; k < interior.size(); ++k) id[interior[k]] = n + (int)k;
    for (int v = 0; v < m; ++v) {
        parent[id[v]] = nd[v].par >= 0 ? id[nd[v].par] : -1;
        age[id[v]] = nd[v].tip >= 0 ? 0.0 : h[v];
    }
    return 0;
}

struct HostTree {
    std::vector<int32_t> left, right, need;
    std::vector<double> e, em;
    int root = -1;
};

// children (lower id first), Sethi-Ullman needs (post-order), branch factors
void host_tree(int n, const int32_t* parent, const double* age, double u, HostTree& t, int model = 0) {
    const int nn = 2 * n - 1;
    t.left.assign(nn, -1);
    t.right.assign(nn, -1);
    t.need.assign(nn, 0);
    t.e.assign(nn, 1.0);
    t.em.assign(nn, 0.0);
    for (int v = 0; v < nn; ++v) {
        const int p = parent[v];
        if (p < 0) { t.root = v; continue; }
        if (t.left[p] < 0) t.left[p] = v;
        else if (v < t.left[p]) { t.right[p] = t.left[p]; t.left[p] = v; }
        else t.right[p] = v;
        branch_data(model, u, age[p] - age[v], t.e[v], t.em[v]);
    }
    // post-order by an explicit stack
    std::vector<int> st;
    std::vector<char> done(nn, 0);
    st.push_back(t.root);
    while (!st.empty()) {
        int v = st.back();
        if (v < n) { st.pop_back(); continue; }
        const int a = t.left[v], b = t.right[v];
        if ((a >= n && !done[a]) || (b >= n && !done[b])) {
            if (a >= n && !done[a]) st.push_back(a);
            if (b >= n && !done[b]) st.push_back(b);
            continue;
        }
        t.need[v] = su_need(a < n ? 0 : t.need[a], b < n ? 0 : t.need[b]);
        done[v] = 1;
        st.pop_back();
    }
}

template <typename ET>
int host_schedule(int n, const HostTree& t, uint32_t* op, ET* e4) {
    std::vector<int> stack(2 * n + 4);
    return emit_schedule(
        n, t.root, [&](int v) { return t.left[v]; }, [&](int v) { return t.right[v]; },
        [&](int v) { return v < n ? 0 : t.need[v]; },
        [&](int i, uint32_t code, int ca, int cb) {
            op[i] = code;
            e4[4 * i + 0] = (ET)t.e[ca];
            e4[4 * i + 1] = (ET)t.em[ca];
            e4[4 * i + 2] = (ET)t.e[cb];
            e4[4 * i + 3] = (ET)t.em[cb];
        },
        stack.data());
}

double host_S(int n, const double* age) {
    // S = sum_k k(k-1) T_k = 2 sum_i (n-i) h_i over sorted coalescence ages (Eq. 18)
    std::vector<double> h(age + n, age + 2 * n - 1);
    std::sort(h.begin(), h.end());
    double S = 0.0;
    for (int i = 1; i <= n - 1; ++i) S += 2.0 * (double)(n - i) * h[i - 1];
    return S;
}

// A, C, G, T -> 0..3 (S2).  With ambiguity codes (f4, S24): IUPAC letters, '-'
// and '?' -> 16 + base-set mask (bit X = base X), else -1.
// fn(i) for i in [0, n), rows spread over up to 32 host threads (alignment ingestion)
template <typename F>
void parallel_rows(int n, F&& fn) {
    const unsigned hw = std::max(1u, std::thread::hardware_concurrency());
    const int nt = (int)std::min<unsigned>({hw, 32u, (unsigned)std::max(1, n)});
    if (nt <= 1) {
        for (int i = 0; i < n; ++i) fn(i);
        return;
    }
    std::vector<std::thread> th;
    for (int t = 0; t < nt; ++t)
        th.emplace_back([&, t] {
            for (int i = t; i < n; i += nt) fn(i);
        });
    for (auto& x : th) x.join();
}

int code_of(char ch, bool ambiguity = false) {
    switch (ch) {
        case 'A': case 'a': return 0;
        case 'C': case 'c': return 1;
        case 'G': case 'g': return 2;
        case 'T': case 't': return 3;
        default: break;
    }
    if (!ambiguity) return -1;
    switch (ch) {
        case 'M': case 'm': return 16 + 3;   // A C
        case 'R': case 'r': return 16 + 5;   // A G
        case 'W': case 'w': return 16 + 9;   // A T
        case 'S': case 's': return 16 + 6;   // C G
        case 'Y': case 'y': return 16 + 10;  // C T
        case 'K': case 'k': return 16 + 12;  // G T
        case 'V': case 'v': return 16 + 7;   // A C G
        case 'H': case 'h': return 16 + 11;  // A C T
        case 'D': case 'd': return 16 + 13;  // A G T
        case 'B': case 'b': return 16 + 14;  // C G T
        case 'N': case 'n': case '-': case '?': return 16 + 15;
        default: return -1;
    }
}

// base set of a code: one bit for A..T, the mask for an ambiguity code
inline int base_set(int code) { return code < 4 ? 1 << code : code - 16; }

// UPGMA (5.1.3 L1287-1295): Hamming distances, average linkage over leaf pairs,
// node height theta0 * d / 2 forced 1e-6 theta0 above the children (S19).
void upgma(int n, int L, const uint8_t* codes, double theta0, int32_t* parent, double* age) {
    const int nn = 2 * n - 1;
    std::vector<std::vector<double>> d(nn, std::vector<double>(nn, 0.0));
    for (int i = 0; i < n; ++i)
        for (int j = i + 1; j < n; ++j) {
            long diff = 0;
            const uint8_t* a = codes + (size_t)i * L;
            const uint8_t* b = codes + (size_t)j * L;
            for (int s = 0; s < L; ++s) diff += (base_set(a[s]) & base_set(b[s])) == 0;  // disjoint sets (S24)
            d[i][j] = d[j][i] = (double)diff;
        }
    std::vector<int> live(n), size(nn, 1);
    for (int i = 0; i < n; ++i) live[i] = i;
    for (int v = 0; v < nn; ++v) { parent[v] = -1; age[v] = 0.0; }
    for (int k = n; k < nn; ++k) {
        // closest pair; ties -> smallest (lower id, higher id) in lexicographic order
        int bi = -1, bj = -1;
        double best = 0.0;
        for (size_t x = 0; x < live.size(); ++x)
            for (size_t y = x + 1; y < live.size(); ++y) {
                int i = std::min(live[x], live[y]), j = std::max(live[x], live[y]);
                double dv = d[i][j];
                if (bi < 0 || dv < best || (dv == best && (i < bi || (i == bi && j < bj)))) {
                    best = dv; bi = i; bj = j;
                }
            }
        double h = theta0 * best / 2.0;
        h = std::max(h, std::max(age[bi], age[bj]) + 1e-6 * theta0);
        age[k] = h;
        parent[bi] = parent[bj] = k;
        size[k] = size[bi] + size[bj];
        std::vector<int> next;
        for (int v : live)
            if (v != bi && v != bj) next.push_back(v);
        for (int v : next) {
            double dv = (size[bi] * d[bi][v] + size[bj] * d[bj][v]) / (double)size[k];
            d[k][v] = d[v][k] = dv;
        }
        next.push_back(k);
        live.swap(next);
    }
}

// Sites per CTA: a multiple of the kernel's exact-sum unit (unit_batches site
// batches; 1..MPCGS_MAXPER = 128 batches), chosen by a small cost model in units of
// one batch: a CTA costs its per-tree setup (schedule compaction, tables:
// ~MPCGS_SETUP batches) plus its batches; the launch takes ceil(CTAs / resident
// CTAs) waves of one CTA.  Few batches per tree and many trees -> one CTA per tree (the
// setup is not repeated per tile); few trees -> more tiles for parallelism.  The
// tree count is the number THIS launch scores (a rank's share of the proposals):
// the site sums are exact (arith.cuh Exact128) over units fixed by the alignment,
// so the tiling never changes a likelihood and every world size gives the same
// chain (P22).
#ifndef MPCGS_MAXPER
#define MPCGS_MAXPER 128
#endif
#ifndef MPCGS_MAXPER_INCR
#define MPCGS_MAXPER_INCR 32
#endif
#ifndef MPCGS_SETUP
#define MPCGS_SETUP 3.0
#endif
void prune_tiling(int n, int L, int ntrees, int precision, int& tiles, int& sites_per_cta, int model = 0) {
    const int batch = prune_batch_sites(n, precision);
    const int unit = prune_unit_batches(n, L, precision);
    const double trees = (double)std::max(ntrees, 1);
    const long batches = (L + batch - 1) / batch;
    const long units = (batches + unit - 1) / unit;
    const double slots = 148.0 * prune_resident_per_sm(n, precision, model != 0);  // resident CTAs
    const long tmin = std::max<long>(1, (units * unit + MPCGS_MAXPER - 1) / MPCGS_MAXPER);
    double best = 1e300;
    long bt = tmin;
    for (long t = tmin; t <= units; ++t) {
        const long per = std::min<long>(((units + t - 1) / t) * unit, batches);  // batches of the largest tile
        const double len = MPCGS_SETUP + (double)per;
        const double ctas = trees * (double)t;
        // a few waves: equal CTAs run in lock-step waves; many: the tail averages out
        // CTAs of one launch have (nearly) equal length and run in lock-step waves: the
        // last, partly empty wave costs a whole CTA (measured: c5 picks 3 tiles of <= 68
        // batches instead of 4 of <= 52, +1.6 %; c5 L = 3e4 +3.5 %)
        const double cost = std::ceil(ctas / slots) * len;
        if (cost < best * (1.0 - 1e-9)) {
            best = cost;
            bt = t;
        }
    }
    tiles = (int)bt;
    sites_per_cta = (int)std::min<long>(((units + bt - 1) / bt) * unit * (long)batch, (long)L);
}

// incremental rescoring (no per-CTA table setup): as many batches per CTA as
// keep >= ~8 CTAs per SM busy, up to MPCGS_MAXPER_INCR.  Each thread multiplies its
// sites over the whole tile before its log, so this tiling depends on the GLOBAL
// proposal count only (identical on every rank: P22); the tile sums are exact.
void incr_tiling(int n, int L, int ntrees_global, int precision, int& tiles, int& sites_per_cta) {
    const int batch = prune_batch_sites(n, precision);
    const long batches = (L + batch - 1) / batch;
    const long want = (long)148 * 8;
    const int per = (int)std::max<long>(1, std::min<long>(MPCGS_MAXPER_INCR, (ntrees_global * batches) / want));
    sites_per_cta = per * batch;
    tiles = (L + sites_per_cta - 1) / sites_per_cta;
}

#ifndef MPCGS_UNIT_MIN_L
#define MPCGS_UNIT_MIN_L 16384
#endif
PruneArgs prune_args(mpcgs_ctx* c, int ntrees, double* out, int out_first, int out_stride) {
    PruneArgs a{};
    a.codes = c->s.codes;
    a.codes2 = c->codes2;
    a.site_w = c->s.site_w;
    a.sum_w = (double)c->L_orig;  // pattern counts sum to the alignment's columns
    // unit-diagonal branches only on long alignments: their per-CTA setup (a log per branch,
    // one more barrier) is paid back over many batches (c5 L = 1e5 +1 %, L <= 3 kbp -1..-3.5 %).
    // A function of the alignment only, so every tiling / world size scores a tree the same way
    a.unit_form = c->L >= MPCGS_UNIT_MIN_L;
    a.W2 = codes2_words(c->L) * (c->s.amb ? 2 : 1);  // 4-bit codes with ambiguity data
    a.Lpad = c->Lpad;
    a.L = c->L;
    a.nops = c->nops;
    for (int i = 0; i < 4; ++i) a.pi[i] = c->s.pi[i];
    a.sched_op = c->s.sched_op;
    a.sched_e = c->s.sched_e;
    a.gm = c->model ? c->s.gm : nullptr;
    a.amb = c->s.amb;
    a.sched_P = c->s.sched_P;
    prune_tiling(c->n, c->L, ntrees, c->precision, a.tiles, a.sites_per_cta, c->model);
    a.unit_batches = prune_unit_batches(c->n, c->L, c->precision);
    a.unit_sites = a.unit_batches * prune_batch_sites(c->n, c->precision);
    a.units = (c->L + a.unit_sites - 1) / a.unit_sites;
    a.tree_need = c->s.tree_need;
    a.tree_acc = c->s.tree_acc;
    a.tile_cnt = c->s.tile_cnt;
    a.out = out;
    a.out_first = out_first;
    a.out_stride = out_stride;
    return a;
}

// enter / leave: order work on the internal stream after the user's stream
mpcgs_status enter(mpcgs_ctx* c) {
    CU(cudaEventRecord(c->ev_a, c->user));
    CU(cudaStreamWaitEvent(c->work, c->ev_a, 0));
    return MPCGS_OK;
}
mpcgs_status leave(mpcgs_ctx* c) {
    CU(cudaStreamSynchronize(c->work));
    return MPCGS_OK;
}

// upload schedules of host trees [first, first+count) and score them into score_out
mpcgs_status score_batch(mpcgs_ctx* c, int count, const int32_t* parent, const double* age, double* out) {
    const int n = c->n, nn = c->nn, nops = c->nops;
    std::vector<uint32_t> ops((size_t)count * nops);
    std::vector<int32_t> needs((size_t)count);
    std::vector<double> e8;
    std::vector<float> e4;
    if (c->precision == 32) e4.resize((size_t)count * nops * 4);
    else e8.resize((size_t)count * nops * 4);
    for (int t = 0; t < count; ++t) {
        std::string why;
        if (check_tree(n, parent + (size_t)t * nn, age + (size_t)t * nn, why))
            return fail(c, MPCGS_E_ARG, "tree " + std::to_string(t) + ": " + why);
        HostTree ht;
        host_tree(n, parent + (size_t)t * nn, age + (size_t)t * nn, c->s.u, ht, c->model);
        int d = c->precision == 32 ? host_schedule<float>(n, ht, ops.data() + (size_t)t * nops,
                                                          e4.data() + (size_t)t * nops * 4)
                                   : host_schedule<double>(n, ht, ops.data() + (size_t)t * nops,
                                                           e8.data() + (size_t)t * nops * 4);
        if (d > c->depth) return fail(c, MPCGS_E_ARG, "tree needs more registers than compiled");
        needs[t] = d;
    }
    CU(cudaMemcpyAsync(c->s.tree_need, needs.data(), 4 * (size_t)count, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.sched_op, ops.data(), ops.size() * 4, cudaMemcpyHostToDevice, c->work));
    if (c->precision == 32)
        CU(cudaMemcpyAsync(c->s.sched_e, e4.data(), e4.size() * 4, cudaMemcpyHostToDevice, c->work));
    else
        CU(cudaMemcpyAsync(c->s.sched_e, e8.data(), e8.size() * 8, cudaMemcpyHostToDevice, c->work));
    PruneArgs a = prune_args(c, count, c->score_out, 0, 1);
    CU(launch_prune(a, count, c->depth, c->precision, c->work));
    CU(cudaMemcpyAsync(out, c->score_out, 8 * (size_t)count, cudaMemcpyDeviceToHost, c->work));
    CU(cudaStreamSynchronize(c->work));
    return MPCGS_OK;
}

mpcgs_status upload_state(mpcgs_ctx* c, const int32_t* parent, const double* age) {
    const int n = c->n, nn = c->nn;
    std::string why;
    if (check_tree(n, parent, age, why)) return fail(c, MPCGS_E_ARG, "generator: " + why);
    HostTree ht;
    host_tree(n, parent, age, c->s.u, ht, c->model);
    if (ht.need[ht.root] > c->depth) return fail(c, MPCGS_E_ARG, "tree needs more registers than compiled");
    double logL = 0.0;
    mpcgs_status st = score_batch(c, 1, parent, age, &logL);
    if (st) return st;
    double gen[2] = {logL, host_S(n, age)};
    CU(cudaMemcpyAsync(c->s.parent, parent, 4 * (size_t)nn, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.left, ht.left.data(), 4 * (size_t)nn, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.right, ht.right.data(), 4 * (size_t)nn, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.need, ht.need.data(), 4 * (size_t)nn, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.age, age, 8 * (size_t)nn, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.e, ht.e.data(), 8 * (size_t)nn, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.em, ht.em.data(), 8 * (size_t)nn, cudaMemcpyHostToDevice, c->work));
    CU(cudaMemcpyAsync(c->s.gen, gen, 16, cudaMemcpyHostToDevice, c->work));
    if (c->incremental) {
        // interior nodes children-first (post-order), then every node's partials
        std::vector<int32_t> order;
        std::vector<int> st{ht.root};
        std::vector<char> done(nn, 0);
        while (!st.empty()) {
            const int v = st.back();
            const int a = ht.left[v], b2 = ht.right[v];
            if ((a >= n && !done[a]) || (b2 >= n && !done[b2])) {
                if (a >= n && !done[a]) st.push_back(a);
                if (b2 >= n && !done[b2]) st.push_back(b2);
                continue;
            }
            done[v] = 1;
            order.push_back(v);
            st.pop_back();
        }
        CU(cudaMemcpyAsync(c->s.gen_order, order.data(), 4 * order.size(), cudaMemcpyHostToDevice, c->work));
        CU(launch_gen_partials(c->s, c->work));
    }
    CU(cudaStreamSynchronize(c->work));
    return MPCGS_OK;
}

mpcgs_status check_status(mpcgs_ctx* c) {
    int64_t st = 0;
    CU(cudaMemcpy(&st, c->s.counters + 2, 8, cudaMemcpyDeviceToHost));
    if (st & STATUS_NUMERIC) return fail(c, MPCGS_E_NUMERIC, "all N+1 weights are non-finite");
    if (st & STATUS_WALK) return fail(c, MPCGS_E_NUMERIC, "resimulation walk did not reach the ancestor");
    return MPCGS_OK;
}

// one step's proposal work for this rank: context, propose, prune
mpcgs_status step_local_launch(mpcgs_ctx* c, uint64_t seed, int64_t step, int N, cudaEvent_t pre = nullptr,
                               cudaEvent_t post = nullptr, bool with_context = true) {
    int first = 1 + c->rank * (N / c->world), count = N / c->world;
    if (with_context) CU(launch_context(c->s, seed, step, c->work));
    CU(launch_propose(c->s, seed, step, first, count, c->work));
    PruneArgs a = prune_args(c, count, c->s.rec, first, REC);
    if (pre) CU(cudaEventRecord(pre, c->work));
    int np = 1;
    if (c->incremental) {
        IncrArgs ia{};
        ia.count = count;
        incr_tiling(c->n, c->L, N, c->precision, ia.tiles, ia.sites_per_cta);
        ia.tree_acc = c->s.tree_acc;
        ia.tile_cnt = c->s.tile_cnt;
        ia.out = c->s.rec;
        ia.out_first = first;
        ia.out_stride = REC;
        CU(launch_score_incr(c->s, ia, c->work));
    } else {
        CU(launch_prune(a, count, c->depth, c->precision, c->work, &np));
    }
    if (post) CU(cudaEventRecord(post, c->work));
    c->launches += (with_context ? 2 : 1) + np;
    return MPCGS_OK;
}

mpcgs_status allgather_records(mpcgs_ctx* c, int N) {
    if (!c->comm) return MPCGS_OK;  // world = 1 without a communicator
    NcclApi& api = nccl();
    const size_t cnt = (size_t)(N / c->world) * REC;
    double* recv = c->s.rec + REC;  // slot 1
    ncclResult_t r = api.allGather(recv + c->rank * cnt, recv, cnt, ncclFloat64, c->comm, c->work);
    if (r != ncclSuccess) return fail(c, MPCGS_E_NCCL, std::string("ncclAllGather: ") + (api.errStr ? api.errStr(r) : "?"));
    return MPCGS_OK;
}

}  // namespace

// ======================================================================== ABI
extern "C" {

const char* mpcgs_version(void) { return "mpcgs-b200 0.1 (sm_100a)"; }

void mpcgs_config_default(mpcgs_config* cfg) {
    if (!cfg) return;
    std::memset(cfg, 0, sizeof(*cfg));
    for (int i = 0; i < 4; ++i) cfg->base_freq[i] = -1.0;
    cfg->mu = 0.0;
    cfg->precision = 64;
    cfg->burnin_steps = 0;
    cfg->max_proposals = 1024;
    cfg->max_samples = 1 << 20;
    cfg->rank = 0;
    cfg->world = 1;
}

size_t mpcgs_workspace_bytes(int32_t n_seq, int32_t n_sites, int32_t max_proposals, int64_t max_samples,
                             int32_t precision) {
    return mpcgs_workspace_bytes_ex(n_seq, n_sites, max_proposals, max_samples, precision, 0);
}

size_t mpcgs_workspace_bytes_ex(int32_t n_seq, int32_t n_sites, int32_t max_proposals, int64_t max_samples,
                                int32_t precision, int32_t incremental) {
    if (n_seq < 2 || n_sites < 1 || max_proposals < 1 || max_samples < 0) return 0;
    return layout(n_seq, n_sites, max_proposals, max_samples, precision, incremental != 0).total;
}

size_t mpcgs_workspace_bytes_cfg(int32_t n_seq, int32_t n_sites, const mpcgs_config* cfg) {
    if (!cfg || n_seq < 2 || n_sites < 1 || cfg->max_proposals < 1 || cfg->max_samples < 0) return 0;
    return layout(n_seq, n_sites, cfg->max_proposals, cfg->max_samples, cfg->precision, cfg->incremental != 0,
                  cfg->model)
        .total;
}

mpcgs_status mpcgs_transition(int32_t model, double kappa, const double* pi, double mu, double t, double* P) {
    if (!pi || !P || !(t >= 0.0) || !std::isfinite(t)) return MPCGS_E_ARG;
    if (model == MPCGS_MODEL_F81) {
        double e, em;
        branch_data(0, mu, t, e, em);
        for (int i = 0; i < 4; ++i)
            for (int j = 0; j < 4; ++j) P[i * 4 + j] = (i == j ? e : 0.0) + em * pi[j];
        return MPCGS_OK;
    }
    if ((model != MPCGS_MODEL_F84 && model != MPCGS_MODEL_HKY85) || !(kappa >= 0.0) || !std::isfinite(kappa))
        return MPCGS_E_ARG;
    for (int i = 0; i < 4; ++i)
        if (!(pi[i] > 0.0)) return MPCGS_E_ARG;
    double Q[16], gm[36];
    rate_matrix(model, kappa, pi, Q);
    eigen_system(Q, pi, gm);
    pmat(gm, t, P);
    return MPCGS_OK;
}

void mpcgs_philox(const uint32_t ctr[4], const uint32_t key[2], uint32_t out[4]) {
    U4 r = philox(U4{ctr[0], ctr[1], ctr[2], ctr[3]}, key[0], key[1]);
    out[0] = r.x;
    out[1] = r.y;
    out[2] = r.z;
    out[3] = r.w;
}

mpcgs_status mpcgs_shard_range(int32_t N, int32_t rank, int32_t world, int32_t* first, int32_t* count) {
    if (N < 1 || world < 1 || rank < 0 || rank >= world || N % world != 0 || !first || !count) return MPCGS_E_ARG;
    *count = N / world;
    *first = 1 + rank * (*count);
    return MPCGS_OK;
}

mpcgs_status mpcgs_upgma(int32_t n, int32_t L, const uint8_t* codes, double theta0, int32_t* parent, double* age) {
    if (n < 2 || L < 0 || !codes || !parent || !age || !(theta0 > 0)) return MPCGS_E_ARG;
    upgma(n, L, codes, theta0, parent, age);
    return MPCGS_OK;
}

int32_t mpcgs_tree_schedule(int32_t n, const int32_t* parent, const double* age, double mu, uint32_t* op,
                            double* e) {
    if (n < 2 || n > MPCGS_MAX_SEQ || !parent || !age || !op || !e) return MPCGS_E_ARG;
    std::string why;
    if (check_tree(n, parent, age, why)) return MPCGS_E_ARG;
    HostTree ht;
    host_tree(n, parent, age, mu, ht);
    return host_schedule<double>(n, ht, op, e);
}

mpcgs_status mpcgs_prune_tiling(int32_t n, int32_t L, int32_t ntrees, int32_t precision, int32_t* tiles,
                                int32_t* sites_per_cta, int32_t* unit_batches) {
    if (n < 3 || n > MPCGS_MAX_SEQ || L < 1 || ntrees < 1 || (precision != 32 && precision != 64)) return MPCGS_E_ARG;
    int t = 0, spc = 0;
    prune_tiling(n, L, ntrees, precision, t, spc);
    if (tiles) *tiles = t;
    if (sites_per_cta) *sites_per_cta = spc;
    if (unit_batches) *unit_batches = prune_unit_batches(n, L, precision);
    return MPCGS_OK;
}

mpcgs_status mpcgs_parse_newick(int32_t n, const char* newick, int32_t* parent, double* age) {
    if (n < 2 || n > MPCGS_MAX_SEQ || !newick || !parent || !age) return MPCGS_E_ARG;
    std::string why;
    std::vector<int32_t> p(2 * (size_t)n - 1);
    std::vector<double> a(2 * (size_t)n - 1);
    if (parse_newick(n, newick, p.data(), a.data(), why) || check_tree(n, p.data(), a.data(), why)) return MPCGS_E_ARG;
    std::copy(p.begin(), p.end(), parent);
    std::copy(a.begin(), a.end(), age);
    return MPCGS_OK;
}

mpcgs_status mpcgs_phylip_dims(const char* path, int32_t* n_seq, int32_t* n_sites) {
    FILE* f = path ? std::fopen(path, "r") : nullptr;
    if (!f) return MPCGS_E_ALIGNMENT;
    int n = 0, L = 0;
    int ok = std::fscanf(f, "%d %d", &n, &L);
    std::fclose(f);
    if (ok != 2 || n < 1 || L < 1) return MPCGS_E_ALIGNMENT;
    *n_seq = n;
    *n_sites = L;
    return MPCGS_OK;
}

mpcgs_status mpcgs_phylip_read(const char* path, char* seqs, int32_t cap) {
    int32_t n, L;
    if (mpcgs_phylip_dims(path, &n, &L) != MPCGS_OK) return MPCGS_E_ALIGNMENT;
    if ((int64_t)n * L > cap) return MPCGS_E_ARG;
    FILE* f = std::fopen(path, "r");
    if (!f) return MPCGS_E_ALIGNMENT;
    std::vector<char> line(1 << 16);
    std::string all;
    {
        int c;
        std::string cur;
        while ((c = std::fgetc(f)) != EOF) all.push_back((char)c);
    }
    std::fclose(f);
    size_t pos = all.find('\n');
    if (pos == std::string::npos) return MPCGS_E_ALIGNMENT;
    ++pos;
    for (int r = 0; r < n; ++r) {
        // skip blank lines
        while (pos < all.size() && (all[pos] == '\n' || all[pos] == '\r')) ++pos;
        size_t eol = all.find('\n', pos);
        if (eol == std::string::npos) eol = all.size();
        std::string ln = all.substr(pos, eol - pos);
        pos = eol + 1;
        // name: first 10 characters, or up to the first blank inside them (S2)
        size_t cut = std::min<size_t>(10, ln.size());
        for (size_t i = 0; i < cut; ++i)
            if (ln[i] == ' ' || ln[i] == '\t') { cut = i; break; }
        std::string rest = ln.substr(cut);
        int got = 0;
        auto eat = [&](const std::string& s) {
            for (char ch : s) {
                if (ch == ' ' || ch == '\t' || ch == '\r') continue;
                if (got >= L) return false;
                if (code_of(ch, true) < 0) return false;  // mpcgs_init decides on ambiguity codes
                seqs[(size_t)r * L + got++] = ch;
            }
            return true;
        };
        if (!eat(rest)) return MPCGS_E_ALIGNMENT;
        while (got < L && pos < all.size()) {  // wrapped sequential format
            eol = all.find('\n', pos);
            if (eol == std::string::npos) eol = all.size();
            std::string more = all.substr(pos, eol - pos);
            pos = eol + 1;
            if (!eat(more)) return MPCGS_E_ALIGNMENT;
        }
        if (got != L) return MPCGS_E_ALIGNMENT;
    }
    return MPCGS_OK;
}

mpcgs_status mpcgs_nccl_unique_id(void* out128) {
    NcclApi& api = nccl();
    if (!api.ok || !out128) return MPCGS_E_NCCL;
    ncclUniqueId id;
    if (api.getUniqueId(&id) != ncclSuccess) return MPCGS_E_NCCL;
    std::memcpy(out128, &id, sizeof(id));
    return MPCGS_OK;
}

// byte codes [n][Lpad] of the flat kernel from the thread-interleaved 2-bit words
// (site k of thread q of a 16-site word at bit (32/si) k + 2 q); padding stays 0
__global__ void k_unpack_codes(const uint32_t* __restrict__ codes2, int W2, int n, int L, int Lpad, int si,
                               uint8_t* __restrict__ out) {
    const long t = (long)blockIdx.x * blockDim.x + threadIdx.x;
    if (t >= (long)n * L) return;
    const int i = (int)(t / L), site = (int)(t - (long)i * L), s16 = site & 15;
    const int shift = (32 / si) * (s16 % si) + 2 * (s16 / si);
    out[(size_t)i * Lpad + site] = (uint8_t)((codes2[(size_t)i * W2 + (site >> 4)] >> shift) & 3u);
}

struct InitTrace {  // MPCGS_TRACE_INIT=1: wall-clock phases of mpcgs_init on stderr
    bool on = std::getenv("MPCGS_TRACE_INIT") != nullptr;
    std::chrono::steady_clock::time_point t = std::chrono::steady_clock::now();
    void mark(const char* what) {
        if (!on) return;
        const auto now = std::chrono::steady_clock::now();
        std::fprintf(stderr, "mpcgs_init %-22s %8.2f ms\n", what, std::chrono::duration<double, std::milli>(now - t).count());
        t = now;
    }
};

mpcgs_status mpcgs_init(const mpcgs_alignment* aln, const mpcgs_config* cfg, double theta0, mpcgs_ctx** out) {
    NvtxRange nvtx_("mpcgs_init");
    InitTrace tr;
    if (!out) return MPCGS_E_ARG;
    *out = nullptr;
    if (!aln || !cfg || !aln->rows) return MPCGS_E_ARG;
    const int n = aln->n_seq;
    int L = aln->n_sites;  // becomes the number of scored sites (patterns) under compression
    if (n < 3 || n > MPCGS_MAX_SEQ || L < 1 || !(theta0 > 0.0) || !std::isfinite(theta0)) return MPCGS_E_ARG;
    if (cfg->precision != 32 && cfg->precision != 64) return MPCGS_E_ARG;
    if (cfg->max_proposals < 1 || cfg->max_proposals > MPCGS_MAX_PROPOSALS || cfg->max_samples < 0) return MPCGS_E_ARG;
    if (cfg->world < 1 || cfg->rank < 0 || cfg->rank >= cfg->world || cfg->burnin_steps < 0) return MPCGS_E_ARG;
    // alignment -> codes (S2: ACGT only; with cfg->ambiguity also IUPAC sets, S24)
    for (int i = 0; i < n; ++i)
        if (!aln->rows[i]) return MPCGS_E_ARG;
    std::vector<uint8_t> codes((size_t)n * L);
    // one table lookup per character, rows in parallel; base counts per row for pi (S1)
    int8_t lut[256];
    for (int ch = 0; ch < 256; ++ch) lut[ch] = (int8_t)code_of((char)ch, cfg->ambiguity != 0);
    std::vector<double> row_cnt((size_t)n * 4, 0.0);
    std::vector<uint8_t> row_bad(n, 0), row_amb(n, 0);
    parallel_rows(n, [&](int i) {
        const unsigned char* src = reinterpret_cast<const unsigned char*>(aln->rows[i]);
        uint8_t* dst = codes.data() + (size_t)i * L;
        long cnt[4] = {0, 0, 0, 0};
        int8_t worst = 0;
        for (int s = 0; s < L; ++s) {
            const int8_t cd = lut[src[s]];
            worst = cd < worst ? cd : worst;
            dst[s] = (uint8_t)cd;
            if (cd >= 0 && cd < 4) ++cnt[cd];
            else if (cd >= 16) row_amb[i] = 1;
        }
        row_bad[i] = worst < 0;
        for (int x = 0; x < 4; ++x) row_cnt[(size_t)i * 4 + x] = (double)cnt[x];
    });
    bool any_amb = false;
    for (int i = 0; i < n; ++i) {
        if (row_bad[i]) return MPCGS_E_ALIGNMENT;
        any_amb |= row_amb[i] != 0;
    }
    tr.mark("codes");
    mpcgs_ctx* c = new mpcgs_ctx();
    c->n = n;
    c->L = L;
    c->nn = 2 * n - 1;
    c->Lpad = (L + 15) & ~15;
    c->nops = n - 1;
    c->depth = prune_depth_for(n);
    c->precision = cfg->precision;
    c->world = cfg->world;
    c->rank = cfg->rank;
    c->burnin = cfg->burnin_steps;
    c->Nmax = cfg->max_proposals;
    c->Mmax = cfg->max_samples;
    c->theta0 = theta0;
    c->user = (cudaStream_t)cfg->stream;
    // model (Eq. 20): pi empirical unless given (S1); u = 1/(1 - sum pi^2) unless given (S3)
    double pi[4];
    bool emp = false;
    for (int i = 0; i < 4; ++i) emp |= cfg->base_freq[i] < 0.0;
    if (emp) {
        double cnt[4] = {0, 0, 0, 0}, known = 0.0;  // ambiguity codes not counted (S24)
        for (int i = 0; i < n; ++i)
            for (int x = 0; x < 4; ++x) {
                cnt[x] += row_cnt[(size_t)i * 4 + x];
                known += row_cnt[(size_t)i * 4 + x];
            }
        for (int i = 0; i < 4; ++i) pi[i] = known > 0.0 ? cnt[i] / known : 0.25;
    } else {
        double sum = 0.0;
        for (int i = 0; i < 4; ++i) { pi[i] = cfg->base_freq[i]; sum += pi[i]; }
        if (!(std::fabs(sum - 1.0) < 1e-9)) { delete c; return MPCGS_E_ARG; }
    }
    double sq = pi[0] * pi[0] + pi[1] * pi[1] + pi[2] * pi[2] + pi[3] * pi[3];
    double u = cfg->mu > 0.0 ? cfg->mu : (sq < 1.0 ? 1.0 / (1.0 - sq) : 1.0);
    // substitution model: F81 unless F84 / HKY85 is asked for
    c->model = cfg->model;
    c->kappa = cfg->kappa;
    double gm[48] = {0};  // eigen-system [0, 36) (flat kernel, k_pmat) + structured constants [36, 41)
    if (c->model != MPCGS_MODEL_F81) {
        const char* why = nullptr;
        if (c->model != MPCGS_MODEL_F84 && c->model != MPCGS_MODEL_HKY85) why = "unknown substitution model";
        else if (!(c->kappa >= 0.0) || !std::isfinite(c->kappa)) why = "kappa must be finite and >= 0";
        else if (!(pi[0] > 0.0 && pi[1] > 0.0 && pi[2] > 0.0 && pi[3] > 0.0)) why = "F84/HKY85 need every pi > 0";
        else if (cfg->incremental) why = "incremental rescoring supports F81 only";
        if (why) {
            c->err = why;
            *out = c;
            return MPCGS_E_ARG;
        }
        double Q[16];
        rate_matrix(c->model, c->kappa, pi, Q);
        eigen_system(Q, pi, gm);
        model_consts(c->model, c->kappa, pi, gm + 36);
        u = 1.0;  // rates normalised to one substitution per unit time (S3); mu is not used
    }
    // G0
    std::vector<int32_t> parent(c->nn);
    std::vector<double> age(c->nn);
    if (cfg->init_newick) {
        std::string why;
        if (parse_newick(n, cfg->init_newick, parent.data(), age.data(), why) ||
            check_tree(n, parent.data(), age.data(), why)) {
            c->err = "init_newick: " + why;
            *out = c;
            return MPCGS_E_ARG;
        }
    } else if (cfg->init_parent && cfg->init_age) {
        std::copy(cfg->init_parent, cfg->init_parent + c->nn, parent.begin());
        std::copy(cfg->init_age, cfg->init_age + c->nn, age.begin());
    } else {
        upgma(n, L, codes.data(), theta0, parent.data(), age.data());
    }
    // device memory
    // site-pattern compression (f3): distinct columns in lexicographic order + counts
    c->L_orig = L;
    std::vector<double> weights;
    int Ls = L;
    if (cfg->compress_patterns) {
        std::vector<int> idx(L);
        for (int s2 = 0; s2 < L; ++s2) idx[s2] = s2;
        auto colcmp = [&](int a2, int b2) {
            for (int i = 0; i < n; ++i) {
                const uint8_t x = codes[(size_t)i * L + a2], y2 = codes[(size_t)i * L + b2];
                if (x != y2) return x < y2;
            }
            return false;
        };
        std::stable_sort(idx.begin(), idx.end(), colcmp);
        std::vector<int> reps;
        for (int k = 0; k < L; ++k) {
            if (k == 0 || colcmp(idx[k - 1], idx[k])) {
                reps.push_back(idx[k]);
                weights.push_back(1.0);
            } else {
                weights.back() += 1.0;
            }
        }
        Ls = (int)reps.size();
        std::vector<uint8_t> comp((size_t)n * Ls);
        for (int i = 0; i < n; ++i)
            for (int k = 0; k < Ls; ++k) comp[(size_t)i * Ls + k] = codes[(size_t)i * L + reps[k]];
        codes.swap(comp);
    }
    L = Ls;
    c->L = L;
    c->Lpad = (L + 15) & ~15;
    c->incremental = cfg->incremental != 0;
    Layout y = layout(n, Ls, c->Nmax, c->Mmax, c->precision, c->incremental, c->model);
    tr.mark("model, G0, layout");
    mpcgs_status st = MPCGS_OK;
    do {
        if (cudaStreamCreateWithFlags(&c->work, cudaStreamNonBlocking) != cudaSuccess ||
            cudaEventCreateWithFlags(&c->ev_a, cudaEventDisableTiming) != cudaSuccess ||
            cudaEventCreate(&c->ev_b) != cudaSuccess) {
            st = fail(c, MPCGS_E_CUDA, "stream/event creation failed (no CUDA device?)");
            break;
        }
        if (cfg->workspace) {
            if (cfg->workspace_bytes < y.total || ((uintptr_t)cfg->workspace & 255)) {
                st = fail(c, MPCGS_E_NOMEM, "workspace too small or not 256-byte aligned");
                break;
            }
            c->ws = cfg->workspace;
            c->ws_bytes = cfg->workspace_bytes;
        } else {
            if (cudaMalloc(&c->ws, y.total) != cudaSuccess) {
                st = fail(c, MPCGS_E_NOMEM, "cudaMalloc of the workspace failed");
                break;
            }
            c->own_ws = true;
            c->ws_bytes = y.total;
        }
        tr.mark("stream, workspace");
        char* b = (char*)c->ws;
        DevState& s = c->s;
        s.n = n; s.nn = c->nn; s.L = L; s.Lpad = c->Lpad; s.nops = c->nops; s.precision = c->precision;
        for (int i = 0; i < 4; ++i) s.pi[i] = pi[i];
        s.u = u;
        s.theta0 = theta0;
        s.codes = (const uint8_t*)(b + y.codes);
        s.parent = (int32_t*)(b + y.parent);
        s.left = (int32_t*)(b + y.left);
        s.right = (int32_t*)(b + y.right);
        s.need = (int32_t*)(b + y.need);
        s.age = (double*)(b + y.age);
        s.e = (double*)(b + y.e);
        s.em = (double*)(b + y.em);
        s.gen = (double*)(b + y.gen);
        s.ctx_i = (int32_t*)(b + y.ctx_i);
        s.ctx_d = (double*)(b + y.ctx_d);
        s.tau = (double*)(b + y.tau);
        s.len = (double*)(b + y.len);
        s.lcnt = (int32_t*)(b + y.lcnt);
        s.entry = (int32_t*)(b + y.entry);
        s.omega = (double*)(b + y.omega);
        s.fixed = (double*)(b + y.fixed);
        s.rec = (double*)(b + y.rec);
        s.tree_need = (int32_t*)(b + y.tree_need);
        s.sched_op = (uint32_t*)(b + y.sched_op);
        s.sched_e = (void*)(b + y.sched_e);
        s.tree_acc = (unsigned long long*)(b + y.tree_acc);
        s.tile_cnt = (uint32_t*)(b + y.tile_cnt);
        s.sS = (double*)(b + y.sS);
        s.sL = (double*)(b + y.sL);
        s.sStep = (int64_t*)(b + y.sStep);
        s.sSlot = (int32_t*)(b + y.sSlot);
        s.counters = (int64_t*)(b + y.counters);
        s.last_draws = (int32_t*)(b + y.last_draws);
        s.theta_buf = (double*)(b + y.theta_buf);
        s.Nmax = c->Nmax;
        s.tiles_max = y.tiles_max;
        s.incremental = c->incremental ? 1 : 0;
        s.GL = c->incremental ? (void*)(b + y.GL) : nullptr;
        s.GE = c->incremental ? (int32_t*)(b + y.GE) : nullptr;
        s.Lg = c->Lpad;
        s.path = (int32_t*)(b + y.path);
        s.pathsib = (int32_t*)(b + y.pathsib);
        s.cpath = (int32_t*)(b + y.cpath);
        s.csib = (int32_t*)(b + y.csib);
        s.ixyz = (int32_t*)(b + y.ixyz);
        s.iee = (double*)(b + y.iee);
        s.cinfo = (int32_t*)(b + y.cinfo);
        s.gen_order = (int32_t*)(b + y.gen_order);
        s.model = c->model ? 1 : 0;
        s.gm = c->model ? (const double*)(b + y.gm) : nullptr;
        s.sched_P = c->model ? (void*)(b + y.sched_P) : nullptr;
        s.Mmax = c->Mmax;
        c->theta_cnt = (unsigned*)(b + y.theta_cnt);
        c->score_out = (double*)(b + y.score_out);
        c->codes2 = (uint32_t*)(b + y.codes2);  // 2-bit base codes, or 4-bit base-set masks (ambiguity data)
        s.amb = any_amb ? 1 : 0;
        s.site_w = cfg->compress_patterns ? (const double*)(b + y.site_w) : nullptr;
        if ((st = enter(c))) break;
        if (cudaMemsetAsync(c->ws, 0, y.total, c->work) != cudaSuccess) { st = fail(c, MPCGS_E_CUDA, "memset"); break; }
        tr.mark("enter, memset");
        // byte codes (the flat kernel) are unpacked on the device from the 2-bit words
        // unless the data hold ambiguity codes (then they are the only codes)
        std::vector<uint8_t> padded(any_amb ? (size_t)n * c->Lpad : 0, 0);
        const int W2 = codes2_words(L), W4 = 2 * W2;
        const int si2 = prune_batch_sites(n, c->precision) / PRUNE_THREADS;  // sites per thread of the table kernel
        std::vector<uint32_t> packed((size_t)n * (any_amb ? W4 : W2), 0u);
        // thread-interleaved order of the table kernel (Codes<SI, BITS>): site k of thread q
        int shift[16], shift4[8];
        for (int s16 = 0; s16 < 16; ++s16) shift[s16] = (32 / si2) * (s16 % si2) + 2 * (s16 / si2);
        for (int s8 = 0; s8 < 8; ++s8) shift4[s8] = (32 / si2) * (s8 % si2) + 4 * (s8 / si2);
        parallel_rows(n, [&](int i) {
            const uint8_t* src = codes.data() + (size_t)i * L;
            if (any_amb) {  // byte codes and 4-bit codes: base-set masks 1..15
                uint8_t* pb = padded.data() + (size_t)i * c->Lpad;
                uint32_t* pw = packed.data() + (size_t)i * W4;
                for (int site = 0; site < L; ++site) {
                    const uint32_t m = (uint32_t)base_set(src[site]);
                    pb[site] = (uint8_t)m;
                    pw[site >> 3] |= m << shift4[site & 7];
                }
                return;
            }
            uint32_t* pw = packed.data() + (size_t)i * W2;
            for (int site = 0; site < L; ++site) pw[site >> 4] |= (uint32_t)src[site] << shift[site & 15];
        });
        if ((any_amb &&
             cudaMemcpyAsync((void*)s.codes, padded.data(), padded.size(), cudaMemcpyHostToDevice, c->work) != cudaSuccess) ||
            (c->codes2 &&
             cudaMemcpyAsync(c->codes2, packed.data(), packed.size() * 4, cudaMemcpyHostToDevice, c->work) != cudaSuccess)) {
            st = fail(c, MPCGS_E_CUDA, "codes upload");
            break;
        }
        if (!any_amb) {
            const long total = (long)n * L;
            k_unpack_codes<<<(unsigned)((total + 255) / 256), 256, 0, c->work>>>(c->codes2, W2, n, L, c->Lpad, si2,
                                                                                 const_cast<uint8_t*>(s.codes));
            if (cudaGetLastError() != cudaSuccess) {
                st = fail(c, MPCGS_E_CUDA, "codes unpack");
                break;
            }
        }
        if (s.gm && cudaMemcpyAsync((void*)s.gm, gm, sizeof(gm), cudaMemcpyHostToDevice, c->work) != cudaSuccess) {
            st = fail(c, MPCGS_E_CUDA, "model upload");
            break;
        }
        if (s.site_w &&
            cudaMemcpyAsync((void*)s.site_w, weights.data(), 8 * weights.size(), cudaMemcpyHostToDevice, c->work) != cudaSuccess) {
            st = fail(c, MPCGS_E_CUDA, "pattern weights upload");
            break;
        }
        tr.mark("pack, upload");
        if ((st = upload_state(c, parent.data(), age.data()))) break;
        tr.mark("upload_state (G0 score)");
        if (cfg->nccl_id) {  // without an id: no communicator (host-staged exchange when world > 1)
            NcclApi& api = nccl();
            if (!api.ok) { st = fail(c, MPCGS_E_NCCL, "NCCL (libnccl.so.2) could not be loaded"); break; }
            ncclUniqueId id;
            std::memcpy(&id, cfg->nccl_id, sizeof(id));
            ncclResult_t r = api.commInitRank(&c->comm, c->world, id, c->rank);
            if (r != ncclSuccess) { st = fail(c, MPCGS_E_NCCL, "ncclCommInitRank failed"); break; }
        }
        st = leave(c);
        tr.mark("nccl, leave");
    } while (0);
    if (st != MPCGS_OK) {
        // keep the context so that mpcgs_last_error can explain; caller frees it
        *out = c;
        return st;
    }
    *out = c;
    return MPCGS_OK;
}

mpcgs_status mpcgs_init_phylip(const char* path, const mpcgs_config* cfg, double theta0, mpcgs_ctx** out) {
    int32_t n, L;
    if (mpcgs_phylip_dims(path, &n, &L) != MPCGS_OK) return MPCGS_E_ALIGNMENT;
    std::vector<char> buf((size_t)n * L);
    mpcgs_status st = mpcgs_phylip_read(path, buf.data(), (int32_t)buf.size());
    if (st) return st;
    std::vector<const char*> rows(n);
    for (int i = 0; i < n; ++i) rows[i] = buf.data() + (size_t)i * L;
    mpcgs_alignment a{n, L, rows.data()};
    return mpcgs_init(&a, cfg, theta0, out);
}

mpcgs_status mpcgs_set_timing(mpcgs_ctx* c, int32_t mode) {
    CHECK_CTX(c);
    c->timing = mode & 3;
    if ((c->timing & 2) && !c->flush_buf) {
        if (cudaMalloc(&c->flush_buf, (size_t)256 << 20) != cudaSuccess)
            return fail(c, MPCGS_E_NOMEM, "flush buffer allocation failed");
    }
    return MPCGS_OK;
}

}  // extern "C"

namespace {
// Enqueue burn-in + sampling on the context's stream (timing mode: run and time
// it); sample_end waits for it.  Loops of several contexts (loci) overlap on the
// device when they are all begun before any is ended.
mpcgs_status sample_end(mpcgs_ctx* c);
// samples stored by the first `k` steps of a run (burn-in draws are not stored; then N
// per step, the last step fewer: Alg. 1, S17)
int64_t stored_after(const mpcgs_ctx* c, int32_t N, int64_t M, int64_t k) {
    const int64_t m = (k - (int64_t)c->burnin) * (int64_t)N;
    return m < 0 ? 0 : (m > M ? M : m);
}

// steps [first, last) of the run (burn-in + ceil(M/N) steps; last < 0 -> to the end).
// first > 0 continues a checkpointed run: the generator (mpcgs_set_state) and the
// samples of steps [0, first) (mpcgs_put_samples) must be in place -- every random
// number is keyed by the global step index, so the continuation is the same chain.
mpcgs_status sample_begin(mpcgs_ctx* c, int32_t N, int64_t M, uint64_t seed, int64_t first = 0,
                          int64_t last = -1) {
    CHECK_CTX(c);
    if (c->pend.active) return fail(c, MPCGS_E_STATE, "a sampling loop is still pending");
    if (N < 1 || N > c->Nmax || N % c->world != 0 || M < 0 || M > c->Mmax)
        return fail(c, MPCGS_E_ARG, "n_proposals / n_samples out of range or not divisible by world");
    if (c->world > 1 && !c->comm)
        return fail(c, MPCGS_E_STATE, "world > 1 without an NCCL id: drive steps with mpcgs_step_local, "
                                      "mpcgs_get_records/put_records and mpcgs_step_finish");
    const int64_t total = (int64_t)c->burnin + (M + N - 1) / N;
    if (last < 0 || last > total) last = total;
    if (first < 0 || first > last) return fail(c, MPCGS_E_ARG, "step range: 0 <= first <= last");
    const int64_t stored0 = stored_after(c, N, M, first);
    if (first > 0 && c->nsamples < stored0)
        return fail(c, MPCGS_E_STATE, "continuing at this step needs the samples of the earlier steps "
                                      "in the store (mpcgs_put_samples)");
    const int64_t steps = total;      // the run's length (k_draw prepares no context past it)
    const int64_t nrun = last - first;  // steps this call runs
    mpcgs_status st = enter(c);
    if (st) return st;
    CU(cudaMemsetAsync(c->s.counters, 0, 8 * 8, c->work));
    if (first > 0) {  // counters[0] = step index, counters[1] = samples stored
        const int64_t cnt[2] = {first, stored0};
        CU(cudaMemcpyAsync(c->s.counters, cnt, sizeof(cnt), cudaMemcpyHostToDevice, c->work));
    }
    c->launches = 0;
    c->prune_ms = c->propose_ms = c->draw_ms = 0.0;
    auto one_step = [&]() -> mpcgs_status {
        mpcgs_status s2 = step_local_launch(c, seed, -1, N, nullptr, nullptr, false);
        if (s2) return s2;
        if ((s2 = allgather_records(c, N))) return s2;
        CU(launch_draw(c->s, seed, -1, N, -1, c->burnin, M, steps, c->work));
        ++c->launches;
        if (c->incremental) {
            CU(launch_commit_incr(c->s, c->work));
            ++c->launches;
        }
        return MPCGS_OK;
    };
    if ((c->timing & 1) && nrun > 0) {
        // device-timed steps: events at step boundaries and around every pruning
        // launch; optional L2 flush between steps, outside the timed intervals
        const size_t need = (size_t)4 * nrun;
        while (c->evpool.size() < need) {
            cudaEvent_t ev;
            CU(cudaEventCreate(&ev));
            c->evpool.push_back(ev);
        }
        for (int64_t k = 0; k < nrun; ++k) {
            if ((c->timing & 2) && c->flush_buf)
                CU(cudaMemsetAsync(c->flush_buf, (int)(k & 0xff), (size_t)256 << 20, c->work));
            CU(cudaEventRecord(c->evpool[4 * k + 0], c->work));
            if (k == 0) {  // the first context; later ones come from k_draw
                CU(launch_context(c->s, seed, -1, c->work));
                ++c->launches;
            }
            if ((st = step_local_launch(c, seed, -1, N, c->evpool[4 * k + 1], c->evpool[4 * k + 2], false))) return st;
            if ((st = allgather_records(c, N))) return st;
            CU(launch_draw(c->s, seed, -1, N, -1, c->burnin, M, steps, c->work));
            ++c->launches;
            if (c->incremental) {
                CU(launch_commit_incr(c->s, c->work));
                ++c->launches;
            }
            CU(cudaEventRecord(c->evpool[4 * k + 3], c->work));
        }
        CU(cudaEventSynchronize(c->evpool[4 * (nrun - 1) + 3]));
        double tot = 0.0, pr = 0.0, pp = 0.0, dr = 0.0;
        for (int64_t k = 0; k < nrun; ++k) {
            float t = 0.f, q = 0.f, p0 = 0.f, d0 = 0.f;
            CU(cudaEventElapsedTime(&t, c->evpool[4 * k + 0], c->evpool[4 * k + 3]));
            CU(cudaEventElapsedTime(&p0, c->evpool[4 * k + 0], c->evpool[4 * k + 1]));
            CU(cudaEventElapsedTime(&q, c->evpool[4 * k + 1], c->evpool[4 * k + 2]));
            CU(cudaEventElapsedTime(&d0, c->evpool[4 * k + 2], c->evpool[4 * k + 3]));
            tot += t;
            pr += q;
            pp += p0;
            dr += d0;
        }
        c->loop_ms = tot;
        c->prune_ms = pr;
        c->propose_ms = pp;
        c->draw_ms = dr;
    } else {
        // CUDA graph of up to graph_steps steps, replayed; the kernels read the step
        // counter from device memory, so one graph serves every step
        const int64_t G = std::min<int64_t>(c->graph_steps, std::max<int64_t>(nrun, 1));
        cudaGraph_t graph = nullptr;
        cudaGraphExec_t exec = nullptr;
        const int64_t reps = nrun / G, rest = nrun % G;
        CU(cudaEventRecord(c->ev_b, c->work));
        CU(launch_context(c->s, seed, -1, c->work));  // the first context; later ones come from k_draw
        c->launches = 1;
        int64_t per_graph = 0;
        if (reps > 0) {
            const int64_t before = c->launches;
            CU(cudaStreamBeginCapture(c->work, cudaStreamCaptureModeThreadLocal));
            for (int64_t k = 0; k < G; ++k) {
                if ((st = one_step())) {
                    cudaStreamEndCapture(c->work, &graph);
                    if (graph) cudaGraphDestroy(graph);
                    return st;
                }
            }
            CU(cudaStreamEndCapture(c->work, &graph));
            CU(cudaGraphInstantiate(&exec, graph, 0));
            per_graph = c->launches - before;
            c->launches = before;
        }
        for (int64_t r = 0; r < reps; ++r) {
            CU(cudaGraphLaunch(exec, c->work));
            c->launches += per_graph;
        }
        for (int64_t k = 0; k < rest; ++k)
            if ((st = one_step())) return st;
        c->pend.graph = graph;
        c->pend.exec = exec;
        CU(cudaEventCreate(&c->pend.end));
        CU(cudaEventRecord(c->pend.end, c->work));
    }
    c->pend.active = true;
    c->pend.N = N;
    c->pend.M = M;
    c->pend.stored = stored_after(c, N, M, last);
    return MPCGS_OK;
}

mpcgs_status sample_end(mpcgs_ctx* c) {
    CHECK_CTX(c);
    if (!c->pend.active) return fail(c, MPCGS_E_STATE, "no sampling loop pending");
    c->pend.active = false;
    mpcgs_status st = MPCGS_OK;
    if (c->pend.end) {
        cudaEvent_t ev_end = c->pend.end;
        c->pend.end = nullptr;
        const cudaError_t e1 = cudaEventSynchronize(ev_end);
        float ms = 0.f;
        const cudaError_t e2 = e1 == cudaSuccess ? cudaEventElapsedTime(&ms, c->ev_b, ev_end) : e1;
        cudaEventDestroy(ev_end);
        if (c->pend.exec) cudaGraphExecDestroy(c->pend.exec);
        if (c->pend.graph) cudaGraphDestroy(c->pend.graph);
        c->pend.exec = nullptr;
        c->pend.graph = nullptr;
        if (e2 != cudaSuccess) return fail(c, MPCGS_E_CUDA, std::string("sampling loop: ") + cudaGetErrorString(e2));
        c->loop_ms = ms;
    }
    if ((st = check_status(c))) return st;
    c->nsamples = c->pend.stored;
    c->lastN = c->pend.N;
    c->sample_theta0 = c->s.theta0;
    return MPCGS_OK;
}
}  // namespace

extern "C" {

mpcgs_status mpcgs_sample(mpcgs_ctx* c, int32_t N, int64_t M, uint64_t seed) {
    NvtxRange nvtx_("mpcgs_sample");
    mpcgs_status st = sample_begin(c, N, M, seed);
    if (st) return st;
    return sample_end(c);
}

mpcgs_status mpcgs_sample_steps(mpcgs_ctx* c, int32_t N, int64_t M, uint64_t seed, int64_t first_step,
                                int64_t last_step) {
    NvtxRange nvtx_("mpcgs_sample_steps");
    mpcgs_status st = sample_begin(c, N, M, seed, first_step, last_step);
    if (st) return st;
    return sample_end(c);
}

mpcgs_status mpcgs_sample_loci(mpcgs_ctx* const* ctxs, int32_t n_loci, int32_t N, int64_t M,
                               const uint64_t* seeds) {
    if (!ctxs || !seeds || n_loci < 1) return MPCGS_E_ARG;
    for (int32_t l = 0; l < n_loci; ++l)
        if (!ctxs[l]) return MPCGS_E_ARG;
    mpcgs_status first = MPCGS_OK;
    int32_t begun = 0;
    for (; begun < n_loci; ++begun) {  // enqueue every locus, then wait for all
        mpcgs_status st = sample_begin(ctxs[begun], N, M, seeds[begun]);
        if (st) { first = st; break; }
    }
    for (int32_t l = 0; l < begun; ++l) {
        mpcgs_status st = sample_end(ctxs[l]);
        if (st && !first) first = st;
    }
    return first;
}


mpcgs_status mpcgs_last_timing_ex(const mpcgs_ctx* c, double* ms4, int64_t* launches) {
    if (!c || !ms4) return MPCGS_E_ARG;
    ms4[0] = c->loop_ms;
    ms4[1] = c->propose_ms;
    ms4[2] = c->prune_ms;
    ms4[3] = c->draw_ms;
    if (launches) *launches = c->launches;
    return MPCGS_OK;
}

mpcgs_status mpcgs_last_timing(const mpcgs_ctx* c, double* loop_ms, double* prune_ms, int64_t* launches) {
    if (!c) return MPCGS_E_ARG;
    if (loop_ms) *loop_ms = c->loop_ms;
    if (prune_ms) *prune_ms = c->prune_ms;
    if (launches) *launches = c->launches;
    return MPCGS_OK;
}

int64_t mpcgs_num_samples(const mpcgs_ctx* c) { return c ? c->nsamples : 0; }

int32_t mpcgs_num_patterns(const mpcgs_ctx* c) { return c ? c->L : 0; }

mpcgs_status mpcgs_get_samples(mpcgs_ctx* c, int64_t first, int64_t count, double* S, double* logL, int64_t* step,
                               int32_t* slot) {
    CHECK_CTX(c);
    if (first < 0 || count < 0 || first + count > c->nsamples) return fail(c, MPCGS_E_ARG, "sample range");
    if (count == 0) return MPCGS_OK;
    if (S) CU(cudaMemcpy(S, c->s.sS + first, 8 * (size_t)count, cudaMemcpyDeviceToHost));
    if (logL) CU(cudaMemcpy(logL, c->s.sL + first, 8 * (size_t)count, cudaMemcpyDeviceToHost));
    if (step) CU(cudaMemcpy(step, c->s.sStep + first, 8 * (size_t)count, cudaMemcpyDeviceToHost));
    if (slot) CU(cudaMemcpy(slot, c->s.sSlot + first, 4 * (size_t)count, cudaMemcpyDeviceToHost));
    return MPCGS_OK;
}

mpcgs_status mpcgs_load_samples(mpcgs_ctx* c, int64_t count, const double* S, const double* logL, double theta0) {
    CHECK_CTX(c);
    if (c->pend.active) return fail(c, MPCGS_E_STATE, "a sampling loop is still pending");
    if (count < 1 || count > c->Mmax || !S) return fail(c, MPCGS_E_ARG, "load_samples: 1 <= count <= max_samples");
    if (!(theta0 > 0.0) || !std::isfinite(theta0)) return fail(c, MPCGS_E_ARG, "load_samples: theta0 must be positive");
    for (int64_t i = 0; i < count; ++i)
        if (!(S[i] >= 0.0) || !std::isfinite(S[i])) return fail(c, MPCGS_E_ARG, "load_samples: S must be finite, >= 0");
    mpcgs_status st = enter(c);
    if (st) return st;
    CU(cudaMemcpyAsync(c->s.sS, S, 8 * (size_t)count, cudaMemcpyHostToDevice, c->work));
    if (logL) CU(cudaMemcpyAsync(c->s.sL, logL, 8 * (size_t)count, cudaMemcpyHostToDevice, c->work));
    else CU(cudaMemsetAsync(c->s.sL, 0, 8 * (size_t)count, c->work));
    CU(cudaMemsetAsync(c->s.sStep, 0xff, 8 * (size_t)count, c->work));
    CU(cudaMemsetAsync(c->s.sSlot, 0xff, 4 * (size_t)count, c->work));
    if ((st = leave(c))) return st;
    c->nsamples = count;
    c->sample_theta0 = theta0;
    return MPCGS_OK;
}

mpcgs_status mpcgs_put_samples(mpcgs_ctx* c, int64_t count, const double* S, const double* logL,
                               const int64_t* step, const int32_t* slot) {
    CHECK_CTX(c);
    if (c->pend.active) return fail(c, MPCGS_E_STATE, "a sampling loop is still pending");
    if (count < 0 || count > c->Mmax || (count > 0 && (!S || !logL)))
        return fail(c, MPCGS_E_ARG, "put_samples: 0 <= count <= max_samples, S and logL given");
    mpcgs_status st = enter(c);
    if (st) return st;
    if (count > 0) {
        CU(cudaMemcpyAsync(c->s.sS, S, 8 * (size_t)count, cudaMemcpyHostToDevice, c->work));
        CU(cudaMemcpyAsync(c->s.sL, logL, 8 * (size_t)count, cudaMemcpyHostToDevice, c->work));
        if (step) CU(cudaMemcpyAsync(c->s.sStep, step, 8 * (size_t)count, cudaMemcpyHostToDevice, c->work));
        else CU(cudaMemsetAsync(c->s.sStep, 0xff, 8 * (size_t)count, c->work));
        if (slot) CU(cudaMemcpyAsync(c->s.sSlot, slot, 4 * (size_t)count, cudaMemcpyHostToDevice, c->work));
        else CU(cudaMemsetAsync(c->s.sSlot, 0xff, 4 * (size_t)count, c->work));
    }
    if ((st = leave(c))) return st;
    c->nsamples = count;
    c->sample_theta0 = c->s.theta0;
    return MPCGS_OK;
}

mpcgs_status mpcgs_score_trees(mpcgs_ctx* c, int32_t n_trees, const int32_t* parent, const double* age,
                               double* logL_out) {
    NvtxRange nvtx_("mpcgs_score_trees");
    CHECK_CTX(c);
    if (n_trees < 0 || (n_trees > 0 && (!parent || !age || !logL_out))) return fail(c, MPCGS_E_ARG, "score_trees args");
    mpcgs_status st = enter(c);
    if (st) return st;
    for (int t0 = 0; t0 < n_trees; t0 += c->Nmax) {
        const int cnt = std::min(c->Nmax, n_trees - t0);
        st = score_batch(c, cnt, parent + (size_t)t0 * c->nn, age + (size_t)t0 * c->nn, logL_out + t0);
        if (st) return st;
    }
    return MPCGS_OK;
}

mpcgs_status mpcgs_set_state(mpcgs_ctx* c, const int32_t* parent, const double* age) {
    CHECK_CTX(c);
    if (!parent || !age) return fail(c, MPCGS_E_ARG, "set_state args");
    mpcgs_status st = enter(c);
    if (st) return st;
    return upload_state(c, parent, age);
}

// checkpoint blob of the chain state: header, then the device generator arrays as
// they are (so a restored chain continues bit for bit: the cached ln P(D|G) and S_G and
// the branch factors the device computed, not host recomputations)
struct StateHeader {
    uint32_t magic, version;
    int32_t n, L_orig, model, precision;
    double theta0;
};
constexpr uint32_t STATE_MAGIC = 0x4b43504du;  // "MPCK"

size_t mpcgs_state_bytes(const mpcgs_ctx* c) {
    return c ? sizeof(StateHeader) + (size_t)c->nn * (4 * 4 + 3 * 8) + 2 * 8 : 0;
}

mpcgs_status mpcgs_save_state(mpcgs_ctx* c, void* buf, size_t bytes) {
    CHECK_CTX(c);
    if (!buf || bytes < mpcgs_state_bytes(c)) return fail(c, MPCGS_E_ARG, "save_state: buffer too small");
    mpcgs_status st = enter(c);
    if (st) return st;
    const size_t nn = (size_t)c->nn;
    StateHeader h{STATE_MAGIC, 1u, c->n, c->L_orig, c->model, c->precision, c->s.theta0};
    unsigned char* p = static_cast<unsigned char*>(buf);
    std::memcpy(p, &h, sizeof(h));
    p += sizeof(h);
    for (int32_t* a : {c->s.parent, c->s.left, c->s.right, c->s.need}) {
        CU(cudaMemcpyAsync(p, a, 4 * nn, cudaMemcpyDeviceToHost, c->work));
        p += 4 * nn;
    }
    for (double* a : {c->s.age, c->s.e, c->s.em}) {
        CU(cudaMemcpyAsync(p, a, 8 * nn, cudaMemcpyDeviceToHost, c->work));
        p += 8 * nn;
    }
    CU(cudaMemcpyAsync(p, c->s.gen, 16, cudaMemcpyDeviceToHost, c->work));
    return leave(c);
}

mpcgs_status mpcgs_load_state(mpcgs_ctx* c, const void* buf, size_t bytes) {
    CHECK_CTX(c);
    if (c->pend.active) return fail(c, MPCGS_E_STATE, "a sampling loop is still pending");
    if (!buf || bytes < mpcgs_state_bytes(c)) return fail(c, MPCGS_E_ARG, "load_state: buffer too small");
    StateHeader h;
    std::memcpy(&h, buf, sizeof(h));
    if (h.magic != STATE_MAGIC || h.version != 1u || h.n != c->n || h.L_orig != c->L_orig || h.model != c->model ||
        h.precision != c->precision || !(h.theta0 > 0.0))
        return fail(c, MPCGS_E_ARG, "load_state: not a checkpoint of this alignment / configuration");
    const size_t nn = (size_t)c->nn;
    const unsigned char* p = static_cast<const unsigned char*>(buf) + sizeof(h);
    std::vector<int32_t> parent(nn), left(nn), right(nn);
    std::memcpy(parent.data(), p, 4 * nn);
    std::memcpy(left.data(), p + 4 * nn, 4 * nn);
    std::memcpy(right.data(), p + 8 * nn, 4 * nn);
    std::vector<double> age(nn);
    std::memcpy(age.data(), p + 16 * nn, 8 * nn);
    std::string why;
    if (check_tree(c->n, parent.data(), age.data(), why)) return fail(c, MPCGS_E_ARG, "load_state: " + why);
    {
        std::vector<int32_t> need(nn);
        std::memcpy(need.data(), p + 12 * nn, 4 * nn);
        for (size_t v = 0; v < nn; ++v)
            if (parent[v] < 0 && need[v] > c->depth)
                return fail(c, MPCGS_E_ARG, "load_state: tree needs more registers than compiled");
    }
    mpcgs_status st = enter(c);
    if (st) return st;
    for (int32_t* a : {c->s.parent, c->s.left, c->s.right, c->s.need}) {
        CU(cudaMemcpyAsync(a, p, 4 * nn, cudaMemcpyHostToDevice, c->work));
        p += 4 * nn;
    }
    for (double* a : {c->s.age, c->s.e, c->s.em}) {
        CU(cudaMemcpyAsync(a, p, 8 * nn, cudaMemcpyHostToDevice, c->work));
        p += 8 * nn;
    }
    CU(cudaMemcpyAsync(c->s.gen, p, 16, cudaMemcpyHostToDevice, c->work));
    c->theta0 = h.theta0;
    c->s.theta0 = h.theta0;
    if (c->incremental) {  // the generator's stored partials (interior nodes children-first)
        const int n = c->n;
        int root = 0;
        for (size_t v = 0; v < nn; ++v)
            if (parent[v] < 0) root = (int)v;
        std::vector<int32_t> order;
        std::vector<int> stk{root};
        std::vector<char> done(nn, 0);
        while (!stk.empty()) {
            const int v = stk.back();
            const int a = left[v], b2 = right[v];
            if ((a >= n && !done[a]) || (b2 >= n && !done[b2])) {
                if (a >= n && !done[a]) stk.push_back(a);
                if (b2 >= n && !done[b2]) stk.push_back(b2);
                continue;
            }
            done[v] = 1;
            order.push_back(v);
            stk.pop_back();
        }
        CU(cudaMemcpyAsync(c->s.gen_order, order.data(), 4 * order.size(), cudaMemcpyHostToDevice, c->work));
        CU(launch_gen_partials(c->s, c->work));
    }
    CU(cudaStreamSynchronize(c->work));
    return leave(c);
}

mpcgs_status mpcgs_get_state(mpcgs_ctx* c, int32_t* parent, double* age, double* logL, double* S) {
    CHECK_CTX(c);
    mpcgs_status st = enter(c);
    if (st) return st;
    double gen[2];
    if (parent) CU(cudaMemcpyAsync(parent, c->s.parent, 4 * (size_t)c->nn, cudaMemcpyDeviceToHost, c->work));
    if (age) CU(cudaMemcpyAsync(age, c->s.age, 8 * (size_t)c->nn, cudaMemcpyDeviceToHost, c->work));
    CU(cudaMemcpyAsync(gen, c->s.gen, 16, cudaMemcpyDeviceToHost, c->work));
    if ((st = leave(c))) return st;
    if (logL) *logL = gen[0];
    if (S) *S = gen[1];
    return MPCGS_OK;
}

mpcgs_status mpcgs_step_local(mpcgs_ctx* c, int64_t step, int32_t N, uint64_t seed) {
    CHECK_CTX(c);
    if (N < 1 || N > c->Nmax || N % c->world != 0 || step < 0) return fail(c, MPCGS_E_ARG, "step_local args");
    mpcgs_status st = enter(c);
    if (st) return st;
    if ((st = step_local_launch(c, seed, step, N))) return st;
    if ((st = leave(c))) return st;
    return check_status(c);
}

mpcgs_status mpcgs_get_records(mpcgs_ctx* c, int32_t first, int32_t count, double* host_rec) {
    CHECK_CTX(c);
    if (first < 0 || count < 0 || first + count > c->Nmax + 1 || (count && !host_rec)) return fail(c, MPCGS_E_ARG, "records range");
    if (!count) return MPCGS_OK;
    mpcgs_status st = enter(c);
    if (st) return st;
    CU(cudaMemcpyAsync(host_rec, c->s.rec + (size_t)first * REC, 8 * REC * (size_t)count, cudaMemcpyDeviceToHost,
                       c->work));
    return leave(c);
}

mpcgs_status mpcgs_put_records(mpcgs_ctx* c, int32_t first, int32_t count, const double* host_rec) {
    CHECK_CTX(c);
    if (first < 1 || count < 0 || first + count > c->Nmax + 1 || (count && !host_rec)) return fail(c, MPCGS_E_ARG, "records range");
    if (!count) return MPCGS_OK;
    // on the work stream, ordered after the caller's stream, and complete on return
    // (a pageable H2D cudaMemcpy may return before the DMA lands)
    mpcgs_status st = enter(c);
    if (st) return st;
    CU(cudaMemcpyAsync(c->s.rec + (size_t)first * REC, host_rec, 8 * REC * (size_t)count, cudaMemcpyHostToDevice,
                       c->work));
    return leave(c);
}

mpcgs_status mpcgs_step_finish(mpcgs_ctx* c, int64_t step, int32_t N, int32_t K, uint64_t seed, int32_t* draws) {
    CHECK_CTX(c);
    if (N < 1 || N > c->Nmax || K < 1 || K > N || step < 0) return fail(c, MPCGS_E_ARG, "step_finish args");
    mpcgs_status st = enter(c);
    if (st) return st;
    CU(cudaMemsetAsync(c->s.counters + 2, 0, 8, c->work));
    CU(launch_draw(c->s, seed, step, N, K, 0, 0, 0, c->work));
    if (c->incremental) CU(launch_commit_incr(c->s, c->work));
    if (draws) CU(cudaMemcpyAsync(draws, c->s.last_draws, 4 * (size_t)K, cudaMemcpyDeviceToHost, c->work));
    if ((st = leave(c))) return st;
    return check_status(c);
}

mpcgs_status mpcgs_step_trace(mpcgs_ctx* c, int64_t step, int32_t N, int32_t K, uint64_t seed, int32_t* target,
                              double* logL, double* S, double* t12, int32_t* pair, int32_t* draws) {
    NvtxRange nvtx_("mpcgs_step_trace");
    CHECK_CTX(c);
    if (c->world != 1) return fail(c, MPCGS_E_STATE, "step_trace needs world = 1 (use step_local/finish)");
    if (N < 1 || N > c->Nmax || K < 1 || K > N || step < 0) return fail(c, MPCGS_E_ARG, "step_trace args");
    mpcgs_status st = enter(c);
    if (st) return st;
    CU(cudaMemsetAsync(c->s.counters + 2, 0, 8, c->work));
    if ((st = step_local_launch(c, seed, step, N))) return st;
    CU(launch_draw(c->s, seed, step, N, K, 0, 0, 0, c->work));
    if (c->incremental) CU(launch_commit_incr(c->s, c->work));
    std::vector<double> rec((size_t)(N + 1) * REC);
    int32_t ci[16];
    CU(cudaMemcpyAsync(rec.data(), c->s.rec, rec.size() * 8, cudaMemcpyDeviceToHost, c->work));
    CU(cudaMemcpyAsync(ci, c->s.ctx_i, sizeof(ci), cudaMemcpyDeviceToHost, c->work));
    if (draws) CU(cudaMemcpyAsync(draws, c->s.last_draws, 4 * (size_t)K, cudaMemcpyDeviceToHost, c->work));
    if ((st = leave(c))) return st;
    if ((st = check_status(c))) return st;
    if (target) *target = ci[0];
    for (int i = 0; i <= N; ++i) {
        const double* r = rec.data() + (size_t)i * REC;
        if (logL) logL[i] = r[0];
        if (S) S[i] = r[1];
        if (t12) { t12[2 * i] = r[2]; t12[2 * i + 1] = r[3]; }
        if (pair) pair[i] = (int32_t)r[4];
    }
    return MPCGS_OK;
}

mpcgs_status mpcgs_set_theta0(mpcgs_ctx* c, double theta0) {
    CHECK_CTX(c);
    if (!(theta0 > 0.0) || !std::isfinite(theta0)) return fail(c, MPCGS_E_ARG, "theta0 must be positive");
    c->theta0 = theta0;
    c->s.theta0 = theta0;
    return MPCGS_OK;
}

mpcgs_status mpcgs_em(mpcgs_ctx* c, int32_t n_iter, int32_t N, int64_t M, uint64_t seed, int32_t G,
                      double* theta_trace) {
    NvtxRange nvtx_("mpcgs_em");
    CHECK_CTX(c);
    if (n_iter < 1 || M < 1) return fail(c, MPCGS_E_ARG, "em: n_iter and n_samples must be positive");
    for (int32_t it = 0; it < n_iter; ++it) {
        mpcgs_status st = mpcgs_sample(c, N, M, seed + (uint64_t)it);
        if (st) return st;
        double th = 0.0;
        if ((st = mpcgs_estimate_theta(c, &th, G, nullptr, nullptr))) return st;
        if (theta_trace) theta_trace[it] = th;
        if ((st = mpcgs_set_theta0(c, th))) return st;
    }
    return MPCGS_OK;
}

mpcgs_status mpcgs_get_model(const mpcgs_ctx* c, double* pi, double* mu) {
    if (!c) return MPCGS_E_ARG;
    if (pi)
        for (int i = 0; i < 4; ++i) pi[i] = c->s.pi[i];
    if (mu) *mu = c->s.u;
    return MPCGS_OK;
}

}  // extern "C"

namespace {
// weighted moments at theta about center (device), returns m0, m1, m2 and the shift used
mpcgs_status moments(mpcgs_ctx* c, double theta, double center, double smin, double smax, double out[4]) {
    const double th0 = c->sample_theta0;
    const double b = 1.0 / theta - 1.0 / th0;
    const double shift = b > 0.0 ? -smin * b : -smax * b;
    double* buf = c->s.theta_buf;
    double* part = buf + 2 * MPCGS_MAX_GRID;
    double* o3 = part + 3 * 296;
    CU(launch_theta_moments(c->s.sS, c->nsamples, th0, theta, shift, center, part, c->theta_cnt, o3, c->work));
    double h[3];
    CU(cudaMemcpyAsync(h, o3, 24, cudaMemcpyDeviceToHost, c->work));
    CU(cudaStreamSynchronize(c->work));
    out[0] = h[0];
    out[1] = h[1];
    out[2] = h[2];
    out[3] = shift;
    return MPCGS_OK;
}

mpcgs_status minmax(mpcgs_ctx* c, double& smin, double& smax) {
    double* o2 = c->s.theta_buf + 2 * MPCGS_MAX_GRID + 3 * 296 + 4;
    CU(launch_minmax(c->s.sS, c->nsamples, o2, c->work));
    double h[2];
    CU(cudaMemcpyAsync(h, o2, 16, cudaMemcpyDeviceToHost, c->work));
    CU(cudaStreamSynchronize(c->work));
    smin = h[0];
    smax = h[1];
    return MPCGS_OK;
}
}  // namespace

extern "C" {

mpcgs_status mpcgs_log_rel_likelihood(mpcgs_ctx* c, double theta, double* out) {
    CHECK_CTX(c);
    if (c->nsamples < 1) return fail(c, MPCGS_E_STATE, "no samples");
    if (!(theta > 0.0) || !out) return fail(c, MPCGS_E_ARG, "theta must be positive");
    mpcgs_status st = enter(c);
    if (st) return st;
    double smin, smax, m[4];
    if ((st = minmax(c, smin, smax))) return st;
    if ((st = moments(c, theta, 0.0, smin, smax, m))) return st;
    *out = (double)(c->n - 1) * std::log(c->sample_theta0 / theta) + m[3] + std::log(m[0]) -
           std::log((double)c->nsamples);
    return MPCGS_OK;
}

}  // extern "C"

namespace {
// theta-hat of one or several loci sharing theta: the joint ln L
// is the sum over loci of Eq. 25 (each locus with its own samples, n and theta0);
// every stationary point solves sum_l S_w,l(theta) = theta sum_l (n_l - 1), so the
// bracket is [sum_l S_min,l, sum_l S_max,l] / sum_l (n_l - 1) (S20).  One locus:
// exactly the single-locus computation.
mpcgs_status estimate_theta_impl(mpcgs_ctx* const* cs, int K, double* theta_hat, int32_t G, double* grid_theta,
                                 double* grid_logL) {
    mpcgs_ctx* c0 = cs[0];
    for (int l = 0; l < K; ++l) {
        CHECK_CTX(cs[l]);
        if (cs[l]->nsamples < 1) return fail(cs[l], MPCGS_E_STATE, "estimate_theta before sample");
        if (cs[l]->pend.active) return fail(cs[l], MPCGS_E_STATE, "a sampling loop is still pending");
    }
    if (!theta_hat || G < 3 || G > MPCGS_MAX_GRID) return fail(c0, MPCGS_E_ARG, "n_grid must be in [3, 4096]");
    std::vector<double> smin(K), smax(K);
    double smin_sum = 0.0, smax_sum = 0.0, dof = 0.0;
    for (int l = 0; l < K; ++l) {
        mpcgs_status st = enter(cs[l]);
        if (st) return st;
        if ((st = minmax(cs[l], smin[l], smax[l]))) return st;
        smin_sum += smin[l];
        smax_sum += smax[l];
        dof += (double)(cs[l]->n - 1);
    }
    if (smin_sum == smax_sum) {  // every stationary point is S/(n-1) (Appendix B)
        *theta_hat = smin_sum / dof;
        for (int g = 0; g < G; ++g) {
            if (grid_theta) grid_theta[g] = *theta_hat;
            if (grid_logL) grid_logL[g] = 0.0;
        }
        return MPCGS_OK;
    }
    const double lo = smin_sum / dof, hi = smax_sum / dof;
    std::vector<double> h(2 * (size_t)G, 0.0), hl(2 * (size_t)G);
    for (int l = 0; l < K; ++l) {  // ln L_l on the common grid, summed over loci
        mpcgs_ctx* c = cs[l];
        double* buf = c->s.theta_buf;
        CU(launch_theta_grid(c->s.sS, c->nsamples, c->n, c->sample_theta0, lo, hi, G, smin[l], smax[l], buf, c->work));
        CU(cudaMemcpyAsync(hl.data(), buf, 16 * (size_t)G, cudaMemcpyDeviceToHost, c->work));
        CU(cudaStreamSynchronize(c->work));
        for (int g = 0; g < G; ++g) {
            h[g] = hl[g];
            h[G + g] += hl[G + g];
        }
    }
    int best = 0;
    for (int g = 1; g < G; ++g)
        if (h[G + g] > h[G + best]) best = g;
    if (grid_theta) std::copy(h.begin(), h.begin() + G, grid_theta);
    if (grid_logL) std::copy(h.begin() + G, h.end(), grid_logL);
    // f(theta) = sum_l (S_w,l - (n_l - 1) theta) has the sign of d lnL / d theta
    auto f_at = [&](double th, double& f, double& fp) -> mpcgs_status {
        double fs = 0.0, vs = 0.0;
        for (int l = 0; l < K; ++l) {
            double m[4];
            const double cen = (double)(cs[l]->n - 1) * th;
            mpcgs_status s2 = moments(cs[l], th, cen, smin[l], smax[l], m);
            if (s2) return s2;
            const double mean = m[1] / m[0];
            fs += mean;  // S_w - c with c = (n-1) theta
            vs += std::max(0.0, m[2] / m[0] - mean * mean);
        }
        f = fs;
        fp = vs / (th * th) - dof;
        return MPCGS_OK;
    };
    // ln L at theta (summed over loci), exact LSE shift
    auto ll = [&](double t, double& v) -> mpcgs_status {
        double tot = 0.0;
        for (int l = 0; l < K; ++l) {
            double m[4];
            mpcgs_status s2 = moments(cs[l], t, 0.0, smin[l], smax[l], m);
            if (s2) return s2;
            tot += (double)(cs[l]->n - 1) * std::log(cs[l]->sample_theta0 / t) + m[3] + std::log(m[0]);
        }
        v = tot;
        return MPCGS_OK;
    };
    // refine the maximum inside the grid cells around grid point b
    auto refine = [&](int b, double& th) -> mpcgs_status {
        mpcgs_status st;
        double blo = b > 0 ? h[b - 1] : lo, bhi = b < G - 1 ? h[b + 1] : hi;
        double flo, fhi, dummy;
        if ((st = f_at(blo, flo, dummy))) return st;
        if ((st = f_at(bhi, fhi, dummy))) return st;
        th = h[b];
        if (flo >= 0.0 && fhi <= 0.0) {  // safeguarded Newton on the stationarity condition
            for (int it = 0; it < 200; ++it) {
                double f, fp;
                if ((st = f_at(th, f, fp))) return st;
                if (f >= 0.0) blo = th;
                else bhi = th;
                double tn = (fp < 0.0) ? th - f / fp : 0.5 * (blo + bhi);
                if (!(tn > blo && tn < bhi)) tn = 0.5 * (blo + bhi);
                if (std::fabs(tn - th) <= 1e-14 * th || bhi - blo <= 1e-15 * bhi) {
                    th = tn;
                    break;
                }
                th = tn;
            }
            return MPCGS_OK;
        }
        // golden-section search on ln L inside the bracket
        const double gr = 0.6180339887498949;
        double a = blo, bb = bhi, x1 = bb - gr * (bb - a), x2 = a + gr * (bb - a), v1, v2;
        if ((st = ll(x1, v1)) || (st = ll(x2, v2))) return st;
        for (int it = 0; it < 200 && bb - a > 1e-15 * bb; ++it) {
            if (v1 > v2) { bb = x2; x2 = x1; v2 = v1; x1 = bb - gr * (bb - a); if ((st = ll(x1, v1))) return st; }
            else { a = x1; x1 = x2; v1 = v2; x2 = a + gr * (bb - a); if ((st = ll(x2, v2))) return st; }
        }
        th = 0.5 * (a + bb);
        return MPCGS_OK;
    };
    // S20: ln L may be bimodal and a coarse grid may rank two close modes wrongly, so
    // every local maximum of the grid curve (up to 4, highest first) is refined and
    // the refined point with the highest ln L is theta-hat (the global argmax)
    std::vector<int> cand;
    for (int g = 0; g < G; ++g) {
        const double v = h[G + g];
        if ((g == 0 || v >= h[G + g - 1]) && (g == G - 1 || v > h[G + g + 1])) cand.push_back(g);
    }
    std::sort(cand.begin(), cand.end(), [&](int a, int b) { return h[G + a] > h[G + b]; });
    if (cand.empty()) cand.push_back(best);
    if (cand.size() > 4) cand.resize(4);
    mpcgs_status st;
    double th = 0.0, th_ll = -INFINITY;
    for (size_t k = 0; k < cand.size(); ++k) {
        double t = 0.0;
        if ((st = refine(cand[k], t))) return st;
        if (cand.size() == 1) {
            th = t;
            break;
        }
        double v;
        if ((st = ll(t, v))) return st;
        if (v > th_ll) {
            th_ll = v;
            th = t;
        }
    }
    *theta_hat = th;
    return MPCGS_OK;
}
}  // namespace

extern "C" {

mpcgs_status mpcgs_estimate_theta(mpcgs_ctx* c, double* theta_hat, int32_t G, double* grid_theta, double* grid_logL) {
    NvtxRange nvtx_("mpcgs_estimate_theta");
    CHECK_CTX(c);
    return estimate_theta_impl(&c, 1, theta_hat, G, grid_theta, grid_logL);
}

mpcgs_status mpcgs_estimate_theta_loci(mpcgs_ctx* const* ctxs, int32_t n_loci, double* theta_hat, int32_t G,
                                       double* grid_theta, double* grid_logL) {
    if (!ctxs || n_loci < 1) return MPCGS_E_ARG;
    for (int32_t l = 0; l < n_loci; ++l)
        if (!ctxs[l]) return MPCGS_E_ARG;
    return estimate_theta_impl(ctxs, n_loci, theta_hat, G, grid_theta, grid_logL);
}

mpcgs_status mpcgs_em_loci(mpcgs_ctx* const* ctxs, int32_t n_loci, int32_t n_iter, int32_t N, int64_t M,
                           const uint64_t* seeds, int32_t G, double* theta_trace) {
    if (!ctxs || !seeds || n_loci < 1 || n_iter < 1 || M < 1) return MPCGS_E_ARG;
    std::vector<uint64_t> sd(n_loci);
    for (int32_t it = 0; it < n_iter; ++it) {
        for (int32_t l = 0; l < n_loci; ++l) sd[l] = seeds[l] + (uint64_t)it;
        mpcgs_status st = mpcgs_sample_loci(ctxs, n_loci, N, M, sd.data());
        if (st) return st;
        double th = 0.0;
        if ((st = mpcgs_estimate_theta_loci(ctxs, n_loci, &th, G, nullptr, nullptr))) return st;
        if (theta_trace) theta_trace[it] = th;
        for (int32_t l = 0; l < n_loci; ++l)
            if ((st = mpcgs_set_theta0(ctxs[l], th))) return st;
    }
    return MPCGS_OK;
}

const char* mpcgs_last_error(const mpcgs_ctx* c) { return c ? c->err.c_str() : "null context"; }

void mpcgs_free(mpcgs_ctx* c) {
    if (!c) return;
    if (c->work) cudaStreamSynchronize(c->work);
    if (c->comm && nccl().ok) nccl().commDestroy(c->comm);
    for (cudaEvent_t e : c->evpool) cudaEventDestroy(e);
    if (c->ev_a) cudaEventDestroy(c->ev_a);
    if (c->ev_b) cudaEventDestroy(c->ev_b);
    if (c->own_ws && c->ws) cudaFree(c->ws);
    if (c->flush_buf) cudaFree(c->flush_buf);
    if (c->work) cudaStreamDestroy(c->work);
    delete c;
}

}  // extern "C"

/*
 * mpcgs.h -- C ABI of the B200 (sm_100a) hot path of the multiple-proposal
 * coalescent genealogy sampler (mpcgs) of P. E. Davis, "Scalable
 * Parallelization of a Markov Coalescent Genealogy Sampler" (2016).
 * Citations "L<a>-<b>" are lines of that paper's PAPER.md; readings S1..S23 are
 * listed in DESIGN.md.
 *
 * The library runs one generalized Metropolis-Hastings (GMH) step per call of
 * its step loop (Alg. 1, Fig. 12):
 *   target draw (4.3 L1079-1093) -> neighbourhood context (4.2 L986-1027) ->
 *   N resimulated proposals (4.2 L1028-1043) -> Felsenstein pruning data
 *   likelihood under F81 (Eq. 19-22) -> weights over N+1 states
 *   (Eq. 29-31) and inverse-CDF draws (L1140-1144),
 * and, after sampling, maximises the relative likelihood L(theta)/L(theta0)
 * (Eq. 25-26, 5.1.5 L1306-1311).
 *
 * Conventions (all entry points):
 *  - Every function returning mpcgs_status returns MPCGS_OK (0) or a negative
 *    code; no C++ exception crosses the ABI.  mpcgs_last_error() describes it.
 *  - Pointers documented "host" are plain host memory owned by the caller,
 *    read or written only during the call.  "device" pointers are CUDA global
 *    memory on the context's device.
 *  - Device memory is the caller's workspace (mpcgs_config.workspace) or, if
 *    that is NULL, memory the context allocates and frees itself.
 *  - MPCGS_E_CUDA and MPCGS_E_NCCL are sticky: after them only mpcgs_free()
 *    and mpcgs_last_error() are valid on that context.
 *  - A context is used by one host thread at a time.  Multi-GPU = one process
 *    (one context) per GPU, ranks given in mpcgs_config.
 *  - Tree arrays: 2n-1 nodes, tips 0..n-1 at age 0, interior nodes n..2n-2,
 *    parent[root] = -1, age[] in mutation units (S22).
 *  - Functions marked [host-only] never touch a GPU and work without one.
 */
#ifndef MPCGS_H
#define MPCGS_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define MPCGS_MAX_SEQ 1024        /* n <= 1024: node ids fit 11 bits, register need <= 10 */
#define MPCGS_MAX_PROPOSALS 4096  /* N per step */
#define MPCGS_MAX_GRID 4096       /* theta grid points */

typedef struct mpcgs_ctx mpcgs_ctx;

typedef enum {
    MPCGS_OK = 0,
    MPCGS_E_ARG = -1,        /* bad argument: n<3, L<1, theta0<=0, N<1, N%world!=0, capacity */
    MPCGS_E_ALIGNMENT = -2,  /* a character outside ACGTacgt (S2) or unreadable PHYLIP */
    MPCGS_E_STATE = -3,      /* call out of order (e.g. estimate before sample) */
    MPCGS_E_CUDA = -4,       /* CUDA runtime error (sticky) */
    MPCGS_E_NCCL = -5,       /* NCCL error or NCCL unavailable for world > 1 (sticky) */
    MPCGS_E_NOMEM = -6,      /* workspace too small / allocation failed */
    MPCGS_E_NUMERIC = -7     /* all N+1 weights non-finite (S6) */
} mpcgs_status;

/* Alignment D (5.1.1 L1229-1241): n rows of L characters in {A,C,G,T,a,c,g,t}.
 * rows: host array of n pointers to L chars each; copied during mpcgs_init. */
typedef struct {
    int32_t n_seq;
    int32_t n_sites;
    const char* const* rows;
} mpcgs_alignment;

typedef struct {
    double base_freq[4];   /* pi (Eq. 20); any entry < 0 -> empirical frequencies over all n*L
                              characters (L702-703, S1) */
    double mu;             /* F81 rate u; <= 0 -> 1/(1 - sum pi^2) (S3), 1 if sum pi^2 == 1 */
    int32_t precision;     /* 64: FP64 partials (parity build) | 32: FP32 partials (fast) */
    int32_t burnin_steps;  /* GMH steps before sampling; 1 draw each, not stored (Fig. 12, S17) */
    int32_t max_proposals; /* capacity: largest N passed to mpcgs_sample (<= MPCGS_MAX_PROPOSALS) */
    int64_t max_samples;   /* capacity: largest M passed to mpcgs_sample */
    const int32_t* init_parent; /* host [2n-1] initial genealogy G0; NULL -> UPGMA (5.1.3, S19) */
    const double* init_age;     /* host [2n-1]; used with init_parent */
    int32_t rank, world;   /* world = 1: one GPU.  world > 1: proposals sharded over ranks */
    const void* nccl_id;   /* host, 128 bytes: ncclUniqueId made by rank 0 with
                              mpcgs_nccl_unique_id() and broadcast by the caller; the library
                              then all-gathers the records with NCCL inside mpcgs_sample (also
                              for world = 1).  NULL with world > 1: no communicator; the caller
                              exchanges records itself (mpcgs_step_local / get_records /
                              put_records / step_finish).  An id serves one communicator:
                              make a fresh one for every context */
    void* stream;          /* cudaStream_t for all work; NULL = the legacy default stream */
    void* workspace;       /* device memory of >= mpcgs_workspace_bytes(...) bytes, 256-B aligned;
                              NULL -> the context allocates (and frees) its own */
    size_t workspace_bytes;
    int32_t incremental;   /* 0: every proposal is scored by full pruning (the paper, 5.2.2).
                              1: incremental rescoring: the generator's partials
                              of all nodes and sites stay in device memory and a proposal
                              recomputes only T, Par and the ancestors of Par (L1390-1398) */
    int32_t compress_patterns; /* 1: score each distinct alignment column once, weighted by its
                              count (exact by site independence, L714-716) */
    int32_t model;         /* substitution model: MPCGS_MODEL_F81 (Eq. 20, the
                              paper's), MPCGS_MODEL_F84 (seq-gen's model of the paper's data,
                              L1508-1510) or MPCGS_MODEL_HKY85.  F84 / HKY85: rates normalised to
                              one expected substitution per unit time (mu is ignored), every
                              pi > 0, incremental = 0 (else MPCGS_E_ARG) */
    double kappa;          /* transition/transversion parameter of F84 / HKY85 (>= 0) */
    int32_t ambiguity;     /* 1: accept IUPAC ambiguity codes (M R W S Y K V H D B N, '-' and '?'
                              as N; either case) as the set of bases they stand for (SURVEY 8(f)
                              f4, reading S24: the tip's partial vector is the set's indicator;
                              empirical pi counts A/C/G/T only; UPGMA counts a site as a
                              difference when the two sets are disjoint).  0: S2, anything but
                              ACGT -> MPCGS_E_ALIGNMENT */
    const char* init_newick; /* host, NUL-terminated Newick G0 (the paper's data come
                              with ms trees, L1499), e.g. "((0:0.1,1:0.1):0.3,2:0.4);": binary,
                              every branch with a length, tips labelled by row index 0..n-1 and
                              contemporaneous (S22, to 1e-5 of the height); copied at init.
                              Takes precedence over init_parent/init_age; NULL -> those or UPGMA.
                              Parse errors -> MPCGS_E_ARG (mpcgs_last_error says where) */
} mpcgs_config;

#define MPCGS_MODEL_F81 0
#define MPCGS_MODEL_F84 1
#define MPCGS_MODEL_HKY85 2

/* [host-only] Fill cfg with defaults: empirical pi, default u, precision 64, burn-in 0,
 * max_proposals 1024, max_samples 1<<20, world 1. */
void mpcgs_config_default(mpcgs_config* cfg);

/* [host-only] Device bytes a context needs for these capacities (full pruning). */
size_t mpcgs_workspace_bytes(int32_t n_seq, int32_t n_sites, int32_t max_proposals,
                             int64_t max_samples, int32_t precision);
/* [host-only] Same, with incremental rescoring on (incremental != 0). */
size_t mpcgs_workspace_bytes_ex(int32_t n_seq, int32_t n_sites, int32_t max_proposals,
                                int64_t max_samples, int32_t precision, int32_t incremental);

/* [host-only] Same, for every capacity / option of cfg (precision, max_proposals,
 * max_samples, incremental, model).  0 on invalid arguments. */
size_t mpcgs_workspace_bytes_cfg(int32_t n_seq, int32_t n_sites, const mpcgs_config* cfg);

/* [host-only] Transition matrix P(t) (row-major, P[i*4+j] = Pr(j at the child | i at the
 * parent), states A,C,G,T) as the kernels form it: F81 by Eq. 20 (L696-699) with rate mu;
 * F84 / HKY85 from the eigen-decomposition of the normalised rate matrix (mu unused).
 * pi: host [4].  MPCGS_E_ARG on a bad model / kappa / t, or pi <= 0 for F84 / HKY85. */
mpcgs_status mpcgs_transition(int32_t model, double kappa, const double* pi, double mu, double t,
                              double* P);

/* Create a context: validate and copy the alignment, compute pi and u, build G0
 * (init_parent/init_age, else UPGMA), upload everything to the device and score
 * P(D|G0) with the pruning kernel.  theta0 > 0 is the driving value (L1239-1241).
 * On an error after allocation *out still receives the context so that
 * mpcgs_last_error() can explain; the caller must mpcgs_free() it. */
mpcgs_status mpcgs_init(const mpcgs_alignment* aln, const mpcgs_config* cfg, double theta0,
                        mpcgs_ctx** out);

/* Same, reading a sequential PHYLIP file (5.1.1 L1233-1237): first line "n L", then
 * per row a name (first 10 characters, or up to the first blank) and L bases. */
mpcgs_status mpcgs_init_phylip(const char* path, const mpcgs_config* cfg, double theta0,
                               mpcgs_ctx** out);

/* Run burn-in then ceil(n_samples / n_proposals) sampling steps with N = n_proposals
 * proposals per step (Alg. 1; Fig. 11/12).  Every random number is Philox4x32-10
 * keyed by `seed` (S21), so results are identical for every world size (P22).
 * Previous samples are discarded.  No host synchronisation inside the loop;
 * returns after the work is complete. */
mpcgs_status mpcgs_sample(mpcgs_ctx* ctx, int32_t n_proposals, int64_t n_samples, uint64_t seed);

/* Checkpoint / resume (long chains): run only steps [first_step, last_step)
 * of the run mpcgs_sample(n_proposals, n_samples, seed) would do (burn-in +
 * ceil(n_samples / n_proposals) steps; last_step < 0 -> to its end).  Every random
 * number is keyed by (seed, global step index) (S21), so a run split at any step
 * boundary is the same chain, bit for bit (tested).  A checkpoint after step k is the
 * chain state (mpcgs_save_state), the samples (mpcgs_get_samples: the first
 * min(max(0, (k - burnin) * N), M) of them), seed, N, M and k; to resume, a context
 * with the same alignment and configuration takes mpcgs_load_state,
 * mpcgs_put_samples, then mpcgs_sample_steps(N, M, seed, k, -1).  first_step > 0
 * with fewer samples stored than the earlier steps drew -> MPCGS_E_STATE; first_step
 * outside [0, last_step] -> MPCGS_E_ARG. */
mpcgs_status mpcgs_sample_steps(mpcgs_ctx* ctx, int32_t n_proposals, int64_t n_samples, uint64_t seed,
                                int64_t first_step, int64_t last_step);

/* theta-hat = argmax L(theta) over the stored samples (Eq. 25-26; S20): a log-spaced
 * grid of n_grid points (3..MPCGS_MAX_GRID) over [S_min, S_max]/(n-1) evaluated on
 * the device, then safeguarded Newton on d lnL/d theta inside the grid cells of every
 * local maximum of the grid curve (up to 4); the refined point of highest ln L wins
 * (L(theta) can be bimodal).
 * grid_theta / grid_logL: host [n_grid] or NULL; grid_logL = ln L(theta). */
mpcgs_status mpcgs_estimate_theta(mpcgs_ctx* ctx, double* theta_hat, int32_t n_grid,
                                  double* grid_theta, double* grid_logL);

/* ln L(theta) (Eq. 25-26) of the stored samples at one theta (device reduction). */
mpcgs_status mpcgs_log_rel_likelihood(mpcgs_ctx* ctx, double theta, double* out);

/* Score arbitrary genealogies with the pruning kernel (Eq. 19-22): host parent/age
 * [n_trees][2n-1] -> host logL_out [n_trees] (ln P(D|G)). */
mpcgs_status mpcgs_score_trees(mpcgs_ctx* ctx, int32_t n_trees, const int32_t* parent,
                               const double* age, double* logL_out);

/* Replace the chain state (generator) by a host tree; its logL is recomputed. */
mpcgs_status mpcgs_set_state(mpcgs_ctx* ctx, const int32_t* parent, const double* age);

/* Checkpoint of the chain state: the generator exactly as the device holds
 * it -- tree arrays, the branch factors and the cached ln P(D|G) and S_G -- plus
 * theta0, behind a header naming the alignment shape and configuration.  The caller
 * owns the host buffer (mpcgs_state_bytes bytes; smaller -> MPCGS_E_ARG).  load_state
 * rejects a blob of another alignment shape / model / precision (MPCGS_E_ARG), sets
 * theta0 and, with incremental rescoring, recomputes the generator's partials.
 * With mpcgs_get_samples / mpcgs_put_samples and mpcgs_sample_steps this resumes a
 * chain bit for bit (set_state would recompute S_G and the branch factors on the
 * host, which may differ from the device's in the last bit). */
size_t mpcgs_state_bytes(const mpcgs_ctx* ctx);
mpcgs_status mpcgs_save_state(mpcgs_ctx* ctx, void* buf, size_t bytes);
mpcgs_status mpcgs_load_state(mpcgs_ctx* ctx, const void* buf, size_t bytes);

/* Read the generator: host parent/age [2n-1]; logL and S (nullable). */
mpcgs_status mpcgs_get_state(mpcgs_ctx* ctx, int32_t* parent, double* age, double* logL,
                             double* S);

/* One GMH step at explicit step index `step` with N proposals and K draws (K <= N),
 * the generator advancing to the last draw; nothing is stored in the sample store.
 * Outputs (host, nullable): target node; per slot 0..N: logL[N+1], S[N+1],
 * t12[(N+1)*2] (new ages of the target and parent ids; slot 0 = generator's),
 * pair[N+1] (0:(c1,c2) 1:(c1,c3) 2:(c2,c3); -1 for slot 0); draws[K]. */
mpcgs_status mpcgs_step_trace(mpcgs_ctx* ctx, int64_t step, int32_t n_proposals, int32_t n_draws,
                              uint64_t seed, int32_t* target, double* logL, double* S,
                              double* t12, int32_t* pair, int32_t* draws);

/* Split GMH step for proposal sharding (S.8(e)): mpcgs_step_local computes this
 * rank's proposal records (slots mpcgs_shard_range) for step `step`;
 * mpcgs_get_records / mpcgs_put_records move records (5 doubles per slot:
 * logL, S, t1, t2, pair) of slots [first, first+count) to / from host memory;
 * mpcgs_step_finish draws K samples from all N+1 records and advances the
 * generator.  With NCCL (world > 1) mpcgs_sample does the exchange itself. */
mpcgs_status mpcgs_step_local(mpcgs_ctx* ctx, int64_t step, int32_t n_proposals, uint64_t seed);
mpcgs_status mpcgs_get_records(mpcgs_ctx* ctx, int32_t first, int32_t count, double* host_rec);
mpcgs_status mpcgs_put_records(mpcgs_ctx* ctx, int32_t first, int32_t count,
                               const double* host_rec);
mpcgs_status mpcgs_step_finish(mpcgs_ctx* ctx, int64_t step, int32_t n_proposals,
                               int32_t n_draws, uint64_t seed, int32_t* draws);

/* Copy samples [first, first+count) to host arrays (each nullable): coalescent
 * statistic S_G = sum k(k-1)T_k (Eq. 18), ln P(D|G), step index, slot index. */
mpcgs_status mpcgs_get_samples(mpcgs_ctx* ctx, int64_t first, int64_t count, double* S,
                               double* logL, int64_t* step, int32_t* slot);
/* Replace the sample store by `count` given samples (1 <= count <= max_samples):
 * host S[count] (S_G >= 0, finite) and logL[count] (nullable -> 0), drawn under the
 * driving value theta0 > 0, for the theta MLE (Eq. 25-26 depend on the samples only
 * through S_G and theta0).  Step and slot indices read back as -1.  Used to test
 * mpcgs_estimate_theta on prescribed sample sets (e.g. S20's bimodal case). */
mpcgs_status mpcgs_load_samples(mpcgs_ctx* ctx, int64_t count, const double* S, const double* logL,
                                double theta0);
/* Restore the sample store of a checkpoint: host S, logL [count] (required when
 * count > 0), step [count] and slot [count] (nullable -> -1).  0 <= count <=
 * max_samples else MPCGS_E_ARG.  The samples count as drawn under the context's
 * current theta0. */
mpcgs_status mpcgs_put_samples(mpcgs_ctx* ctx, int64_t count, const double* S, const double* logL,
                               const int64_t* step, const int32_t* slot);
int64_t mpcgs_num_samples(const mpcgs_ctx* ctx);
/* Sites the kernels score: distinct columns with compress_patterns, else n_sites. */
int32_t mpcgs_num_patterns(const mpcgs_ctx* ctx);

/* Re-drive: theta0 <- theta (L791-797).  Cached P(D|G) stays valid (Eq. 23). */
mpcgs_status mpcgs_set_theta0(mpcgs_ctx* ctx, double theta0);

/* EM loop of Fig. 11 (L1208-1225, L791-797): n_iter times { burn-in + sample
 * (n_proposals, n_samples, seed + it); theta-hat over a n_grid grid;
 * theta0 <- theta-hat }.  theta_trace: host [n_iter] (nullable) receives each
 * iteration's estimate; the chain state carries over between iterations. */
mpcgs_status mpcgs_em(mpcgs_ctx* ctx, int32_t n_iter, int32_t n_proposals, int64_t n_samples,
                      uint64_t seed, int32_t n_grid, double* theta_trace);

/* Multiple loci: loci have independent genealogies and share theta, so
 * the joint relative likelihood is the product over loci of Eq. 25 (L765-797).  ctxs: host
 * array of n_loci contexts (one per locus alignment; any n, L, model; same device).
 *
 * mpcgs_sample_loci: mpcgs_sample on every locus with seeds[l] (host [n_loci]); all loops are
 * enqueued (each on its context's stream) before any is waited for, so loci overlap on the GPU.
 * Returns the first error; every enqueued loop is finished.
 * mpcgs_estimate_theta_loci: the global argmax of sum_l ln L_l(theta) over the bracket
 * [sum_l S_min,l, sum_l S_max,l] / sum_l (n_l - 1) (S20 generalised), grid of n_grid points
 * (grid_theta / grid_logL: host [n_grid], nullable; grid_logL is the summed curve) then
 * safeguarded Newton on sum_l (S_w,l(theta) - (n_l - 1) theta).  One locus = mpcgs_estimate_theta.
 * mpcgs_em_loci: n_iter times { sample_loci(seeds[l] + it); joint theta-hat; every theta0 <- it }.
 * MPCGS_E_ARG on null / empty arrays; MPCGS_E_STATE if a locus has no samples. */
mpcgs_status mpcgs_sample_loci(mpcgs_ctx* const* ctxs, int32_t n_loci, int32_t n_proposals,
                               int64_t n_samples, const uint64_t* seeds);
mpcgs_status mpcgs_estimate_theta_loci(mpcgs_ctx* const* ctxs, int32_t n_loci, double* theta_hat,
                                       int32_t n_grid, double* grid_theta, double* grid_logL);
mpcgs_status mpcgs_em_loci(mpcgs_ctx* const* ctxs, int32_t n_loci, int32_t n_iter,
                           int32_t n_proposals, int64_t n_samples, const uint64_t* seeds,
                           int32_t n_grid, double* theta_trace);

/* Model parameters actually used (host out: pi[4], u). */
mpcgs_status mpcgs_get_model(const mpcgs_ctx* ctx, double* pi, double* mu);

/* Timing mode for mpcgs_sample: on -> CUDA events bracket every pruning launch
 * (and the loop runs as plain launches, not a CUDA graph). */
mpcgs_status mpcgs_set_timing(mpcgs_ctx* ctx, int32_t on);

/* Device time (ms) of the last mpcgs_sample loop and of its pruning launches
 * (CUDA events on the context stream), and kernel launches it issued. */
mpcgs_status mpcgs_last_timing(const mpcgs_ctx* ctx, double* loop_ms, double* prune_ms,
                               int64_t* launches);

/* Per-phase device times (ms) of the last device-timed mpcgs_sample loop (timing mode bit 0),
 * summed over its steps, from the same CUDA events: ms4[0] the loop, [1] context + proposal
 * resimulation (k_context / k_propose), [2] pruning, [3] record exchange + weights/draws/commit
 * (k_draw, k_commit_incr).  ms4: host [4]; launches nullable. */
mpcgs_status mpcgs_last_timing_ex(const mpcgs_ctx* ctx, double* ms4, int64_t* launches);

/* [measurement] Microbenchmarked peak of this GPU for the roofline of the ALU-bound pruning
 * kernels: kind 0 = FP64 FMA throughput (TFLOP/s, FMA = 2 flops), 1 = FP32 FMA
 * (TFLOP/s), 2 = shared-memory load bandwidth (GB/s, ld.shared.v4).  Best of 5 launches of
 * 8 CTAs x 256 threads per SM on the current device, timed with CUDA events (~5 ms each).
 * No context needed.  MPCGS_E_ARG on a bad kind or NULL value. */
mpcgs_status mpcgs_probe_peak(int32_t kind, double* value);

const char* mpcgs_last_error(const mpcgs_ctx* ctx);
void mpcgs_free(mpcgs_ctx* ctx);

/* ---------------------------------------------------------------- host-only helpers */
/* [host-only] Proposal slots owned by `rank`: slots first..first+count-1 of 1..N. */
mpcgs_status mpcgs_shard_range(int32_t n_proposals, int32_t rank, int32_t world, int32_t* first,
                               int32_t* count);
/* [host-only] UPGMA G0 (5.1.3 L1287-1295, S19) from codes[n][L] in {0..3}, or 16 + base-set
 * mask for an ambiguity code (S24: a site differs when the two sets are disjoint). */
mpcgs_status mpcgs_upgma(int32_t n_seq, int32_t n_sites, const uint8_t* codes, double theta0,
                         int32_t* parent, double* age);
/* [host-only] Site tiling of one pruning launch scoring `ntrees` genealogies (a rank's
 * share of the proposals): tiles x sites_per_cta sites per genealogy, and the exact-sum
 * unit in site batches.  The tiling follows ntrees; the
 * likelihoods do not (site sums are exact over units fixed by n, L and precision, P22).
 * Outputs nullable; MPCGS_E_ARG on n < 3, L < 1, ntrees < 1 or a bad precision. */
mpcgs_status mpcgs_prune_tiling(int32_t n_seq, int32_t n_sites, int32_t ntrees, int32_t precision,
                                int32_t* tiles, int32_t* sites_per_cta, int32_t* unit_batches);
/* [host-only] Parse a Newick genealogy of n_seq tips (grammar and rules of
 * mpcgs_config.init_newick) into parent/age [2n-1] host arrays: interior ids n..2n-2 in
 * ascending age (ties: post-order), a node's age = its longest path down to a tip.
 * MPCGS_E_ARG on any syntax / shape / label / ultrametricity error. */
mpcgs_status mpcgs_parse_newick(int32_t n_seq, const char* newick, int32_t* parent, double* age);
/* [host-only] Post-order register schedule of a tree as used by the pruning kernel
 * (DESIGN.md "prune"): op[i] = type | sp<<2 | tipA<<6 | tipB<<17, e[2i], e[2i+1] branch
 * factors exp(-u t); returns the register need (max stack depth) or < 0 on error. */
int32_t mpcgs_tree_schedule(int32_t n_seq, const int32_t* parent, const double* age, double mu,
                            uint32_t* op, double* e);
/* [host-only] Sequential PHYLIP reader: dims, then rows (n*L chars, row-major).  Accepts ACGT
 * and the IUPAC ambiguity characters (mpcgs_init rejects the latter unless cfg->ambiguity);
 * anything else -> MPCGS_E_ALIGNMENT. */
mpcgs_status mpcgs_phylip_dims(const char* path, int32_t* n_seq, int32_t* n_sites);
mpcgs_status mpcgs_phylip_read(const char* path, char* seqs, int32_t cap_chars);
/* [host-only] Philox4x32-10 block (for known-answer checks of the device generator). */
void mpcgs_philox(const uint32_t ctr[4], const uint32_t key[2], uint32_t out[4]);
/* [host-only] A fresh ncclUniqueId (128 bytes) via the dynamically loaded NCCL. */
mpcgs_status mpcgs_nccl_unique_id(void* out128);
const char* mpcgs_version(void);

#ifdef __cplusplus
}
#endif
#endif

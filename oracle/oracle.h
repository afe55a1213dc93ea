/*
 * oracle.h -- plain, slow, FP64 CPU oracle of the mpcgs hot path.
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and
 * bench.py's cpu_baseline / --impl reference legs may load this library.
 * It shares no code, header, table or constant generator with the CUDA
 * library under paper_conf_ipps_davistzw17_b200/ (and vice versa).
 *
 * Every function cites the passage of PAPER.md (P. E. Davis, "Scalable
 * Parallelization of a Markov Coalescent Genealogy Sampler", 2016) it follows,
 * as "L<a>-<b> (section / equation)".  Where the paper is silent or garbled
 * the reading is the one listed in DESIGN.md "Readings" (S1..S23, after
 * SURVEY.md section 8(c)).
 *
 * Tree representation (all functions): 2n-1 nodes; tips 0..n-1 (age 0),
 * interior nodes n..2n-2; parent[root] = -1; age[] in coalescent time units
 * (mutation units, S22).  Children of a node are ordered by ascending id.
 *
 * Tip data: codes[tip*L + site] in {0,1,2,3} = {A,C,G,T}, or 16 + m for an
 * ambiguity code whose base set is the 4-bit mask m (bit X = base X; 16 + 15 = N;
 * SURVEY 8(f) f4, reading S24).
 */
#ifndef MPCGS_ORACLE_H
#define MPCGS_ORACLE_H
#include <stdint.h>

#define ORC_TAG_TARGET 0u
#define ORC_TAG_PROPOSE 1u
#define ORC_TAG_DRAW 2u

#define ORC_OK 0
#define ORC_E_ARG -1
#define ORC_E_TREE -2
#define ORC_E_NUMERIC -7

/* RNG (reading S21 / SURVEY 8(c) c7) */
void orc_philox4x32_10(const uint32_t ctr[4], const uint32_t key[2], uint32_t out[4]);
double orc_u01(uint32_t w0, uint32_t w1);
double orc_uniform(uint64_t seed, uint32_t c1, uint32_t step, uint32_t tag, uint32_t idx);

/* F81 model (Eq. 20; readings S1, S3) */
void orc_base_freqs(int n, int L, const uint8_t* codes, double pi[4]);
double orc_default_rate(const double pi[4]);
void orc_transition(double t, double u, const double pi[4], double P[16]);

/* Model variants (seq-gen's F84 of the paper's data, L1508-1510,
 * L1531-1533): model 0 = F81 (Eq. 20), 1 = F84, 2 = HKY85, transition /
 * transversion parameter kappa; rates normalised to one expected substitution
 * per unit time (reading S3).  Closed forms; states A, C, G, T = 0..3, purines
 * {A, G}, pyrimidines {C, T}. */
double orc_model_rate(int model, double kappa, const double pi[4]);
void orc_transition_model(int model, double kappa, double t, const double pi[4], double P[16]);
double orc_log_likelihood_model(int model, double kappa, int n, int L, const uint8_t* codes,
                                const int32_t* parent, const double* age, const double pi[4],
                                double* site_ll);

/* Tree checks */
int orc_check_tree(int n, const int32_t* parent, const double* age);

/* Data likelihood P(D|G): Eq. 19-22 (L660-719) evaluated in log space (5.3, Eq. 32) */
double orc_log_likelihood(int n, int L, const uint8_t* codes, const int32_t* parent,
                          const double* age, const double pi[4], double u, double* site_ll);

/* Coalescent prior (Eq. 17-18) */
double orc_coalescent_S(int n, const double* age);
double orc_log_prior(int n, const double* age, double theta);

/* Target draw (4.3 L1079-1093; reading S7) */
int orc_pick_target(int n, const int32_t* parent, uint64_t seed, uint32_t step);

/* Neighbourhood context (4.2 L986-1027); info = {T,Par,A,rootcase,k0,m,c0,c1,c2} */
int orc_context_info(int n, const int32_t* parent, const double* age, double theta0, int target,
                     int32_t* info, double* tau, double* len, int32_t* l, int32_t* entry,
                     double* omega, double* beta);

/* One LAMARC resimulation (4.2 L1028-1043) in the neighbourhood of `target` */
int orc_propose(int n, const int32_t* parent, const double* age, double theta0, int target,
                uint64_t seed, uint32_t step, uint32_t slot, int32_t* new_parent,
                double* new_age, double* t12, int32_t* pair, int32_t* flag);

/* Weights over the N+1 states (Eq. 29-31) and inverse-CDF draws (L1140-1144) */
int orc_weights(int nslots, const double* logL, double* w, double* cum);
int orc_draw(int nslots, const double* cum, double u, int32_t* flag);

/* One generalized Metropolis-Hastings step (Alg. 1, Fig. 12) */
int orc_gmh_step(int n, int L, const uint8_t* codes, const double pi[4], double u,
                 double theta0, int N, int K, uint64_t seed, uint32_t step,
                 int32_t* gen_parent, double* gen_age, double* gen_logL,
                 int32_t* out_target, double* slot_logL, double* slot_S, double* slot_t12,
                 int32_t* slot_pair, int32_t* slot_flag, int32_t* draws, int32_t* draw_flag);

/* Same step with P(D|G) under model 1 (F84) / 2 (HKY85), kappa */
int orc_gmh_step_model(int model, double kappa, int n, int L, const uint8_t* codes,
                       const double pi[4], double theta0, int N, int K, uint64_t seed,
                       uint32_t step, int32_t* gen_parent, double* gen_age, double* gen_logL,
                       int32_t* out_target, double* slot_logL, double* slot_S, double* slot_t12,
                       int32_t* slot_pair, int32_t* slot_flag, int32_t* draws, int32_t* draw_flag);

/* Burn-in + sampling chain (Fig. 11/12, Alg. 1) */
int orc_run_chain(int n, int L, const uint8_t* codes, const double pi[4], double u,
                  double theta0, int N, int burnin, int M, uint64_t seed,
                  int32_t* gen_parent, double* gen_age, double* S_out, double* logL_out,
                  int64_t* step_out, int32_t* slot_out, int32_t* n_flagged,
                  int64_t* first_flag_step);
/* EM re-drive (Fig. 11) */
int orc_em(int n, int L, const uint8_t* codes, const double pi[4], double u, double theta0,
           int N, int burnin, int M, uint64_t seed, int n_iter, int G, int32_t* gen_parent,
           double* gen_age, double* theta_trace, int64_t* first_flag);

/* Relative likelihood and MLE (Eq. 25-26; 5.1.5; Alg. 2; reading S20) */
double orc_log_rel_likelihood(int M, const double* S, int n, double theta0, double theta);
double orc_weighted_mean_S(int M, const double* S, double theta0, double theta);
double orc_em_map(int M, const double* S, int n, double theta0, double theta);
double orc_theta_hat(int M, const double* S, int n, double theta0, int G,
                     double* grid_theta, double* grid_ll);
/* Multiple loci sharing theta: product of Eq. 25 over loci; samples
   of locus l at S[sum_{k<l} M_k ...] */
double orc_log_rel_likelihood_loci(int K, const int* M, const double* S, const int* n,
                                   const double* theta0, double theta);
double orc_theta_hat_loci(int K, const int* M, const double* S, const int* n,
                          const double* theta0, int G, double* grid_theta, double* grid_ll);
double orc_theta_alg2(int M, const double* S, int n, double theta0, int max_iter);

/* Initial genealogy G0 by UPGMA (5.1.3 L1287-1295; reading S19) */
int orc_upgma(int n, int L, const uint8_t* codes, double theta0, int32_t* parent, double* age);

#endif

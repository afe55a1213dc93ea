// kernels.cuh -- launch interfaces of the device kernels (internal to the library).
#pragma once
#include <cuda_runtime.h>

#include "common.cuh"

namespace mpcgs {

constexpr int PRUNE_THREADS = 128;
#ifndef MPCGS_SI64
#define MPCGS_SI64 4
#endif
#ifndef MPCGS_SI32
#define MPCGS_SI32 4
#endif
#ifndef MPCGS_DR
#define MPCGS_DR 3
#endif
constexpr int PRUNE_SI64 = MPCGS_SI64;  // sites interleaved per thread, FP64 partials
constexpr int PRUNE_SI32 = MPCGS_SI32;  // FP32 partials
constexpr int PRUNE_DR = MPCGS_DR;      // register-resident stack levels (deeper ones spill to shared memory)
constexpr int PRUNE_SPILL = 2; // shared-memory stack levels; trees needing more use the flat kernel

struct PruneArgs {
    const uint8_t* codes;       // [n][Lpad] bytes (flat kernel)
    const uint32_t* codes2;     // [n][W2] 2-bit packed, 16 sites per word (table kernel)
    int Lpad, L, nops, W2;
    double pi[4];
    const uint32_t* sched_op;  // [ntrees][nops]
    const void* sched_e;       // [ntrees][nops] float4 / double4
    const double* gm;          // general model (f4): [36] eigen-system of Q, else nullptr (F81)
    void* sched_P;             // general model: [ntrees][nops][32] P matrices (float / double)
    int amb;                   // base-set codes (ambiguity, S24): byte masks (flat kernel), 4-bit codes2 (tables)
    // site tiles: tile t covers exact-sum units [t*units/tiles, (t+1)*units/tiles) of
    // unit_sites sites each (balanced; tile_range below); sites_per_cta = the largest tile
    int tiles, sites_per_cta, units, unit_sites;
    const double* site_w;      // [L] pattern counts (compressed sites, f3) or nullptr
    double sum_w;              // sum of the site weights (= alignment columns)
    int unit_form;             // FP64 table kernel: unit-diagonal branches allowed (a function of the alignment only)
    const int32_t* tree_need;  // [ntrees] register need of each tree's schedule (nullable)
    int need_cap;              // set by launch_prune: largest need the table kernel serves
    int trip_cap;              // set by launch_prune: fused triplets per tree (table kernel)
    int code_bufs;             // set by launch_prune: tip-code staging buffers of the table kernel (1 or 2)
    int unit_batches;          // table kernel: site batches per exact-sum unit (tiles hold whole units)
    unsigned long long* tree_acc;  // [ntrees][4] exact site-sum accumulators (Exact128), zero on entry
    uint32_t* tile_cnt;        // [ntrees], zero on entry, reset by the kernel
    double* out;               // logL of tree t -> out[(out_first + t) * out_stride]
    int out_first, out_stride;
};
__device__ __forceinline__ void tile_range(const PruneArgs& a, int tile, int& s_begin, int& s_end) {
    const int u0 = (int)(((long long)tile * a.units) / a.tiles);
    const int u1 = (int)(((long long)(tile + 1) * a.units) / a.tiles);
    s_begin = u0 * a.unit_sites;
    s_end = min(a.L, u1 * a.unit_sites);
}
constexpr int FLAT_UNIT_SITES = 256;  // flat kernel: sites per exact-sum unit (tiles hold whole units)
// site batches per exact-sum unit of the table kernel: a function of the alignment
// only (never of the number of proposals or ranks), so that every tiling a rank may
// choose sums the same terms (P22)
int prune_unit_batches(int n, int L, int precision);

int prune_depth_for(int n);
int prune_max_need(int n);
int prune_need_cap(int n);
int prune_batch_sites(int n, int precision);  // sites_per_cta must be a multiple of this
bool prune_uses_tables(int n, int precision, bool general_model = false, bool amb = false);
int prune_resident_per_sm(int n, int precision, bool general_model = false);  // tiling cost model
cudaError_t launch_prune(const PruneArgs& a, int ntrees, int depth, int precision, cudaStream_t st,
                         int* n_launched = nullptr);

// step kernels (step.cu); step < 0 -> read the step index from counters[0]
cudaError_t launch_context(const DevState& s, uint64_t seed, int64_t step, cudaStream_t st);
cudaError_t launch_propose(const DevState& s, uint64_t seed, int64_t step, int slot_first, int count,
                           cudaStream_t st);
// draw: K < 0 -> loop mode (burn-in / sampling from counters, store, advance step)
// loop mode also computes the context of step+1 when step+1 < total_steps
cudaError_t launch_draw(const DevState& s, uint64_t seed, int64_t step, int N, int K, int burnin,
                        int64_t M, int64_t total_steps, cudaStream_t st);
cudaError_t launch_fill_gen_record(const DevState& s, cudaStream_t st);

// incremental rescoring (incr.cu)
struct IncrArgs {
    int count;                 // proposals of this rank (local slots 0..count-1)
    int tiles, sites_per_cta;
    unsigned long long* tree_acc;  // [count][4] exact site-sum accumulators
    uint32_t* tile_cnt;        // [count]
    double* out;               // logL of local proposal t -> out[(out_first + t) * out_stride]
    int out_first, out_stride;
};
cudaError_t launch_gen_partials(const DevState& s, cudaStream_t st);
cudaError_t launch_commit_incr(const DevState& s, cudaStream_t st);
cudaError_t launch_score_incr(const DevState& s, const IncrArgs& a, cudaStream_t st);

// theta kernels (theta.cu)
cudaError_t launch_minmax(const double* S, int64_t M, double* out2, cudaStream_t st);
cudaError_t launch_theta_grid(const double* S, int64_t M, int n, double theta0, double lo, double hi, int G,
                              double smin, double smax, double* out, cudaStream_t st);
cudaError_t launch_theta_moments(const double* S, int64_t M, double theta0, double theta, double shift,
                                 double center, double* part, unsigned* cnt, double* out3,
                                 cudaStream_t st);

}  // namespace mpcgs

// prune.cu -- host-side routing of the pruning launches (kernels and launch
// templates in prune_kernels.cuh; one translation unit per precision x model:
// prune_f64.cu, prune_f32.cu, prune_f64_gm.cu, prune_f32_gm.cu).
#include "prune_kernels.cuh"

namespace mpcgs {

int prune_depth_for(int n) {
    int d = 0;
    while ((2 << d) <= n) ++d;  // floor(log2 n) = max Sethi-Ullman need of an n-tip tree
    if (d <= 4) return 4;
    if (d <= 6) return 6;
    if (d <= 8) return 8;
    return 10;
}

int prune_max_need(int n) {
    int d = 0;
    while ((2 << d) <= n) ++d;
    return d < 1 ? 1 : d;
}

// sites interleaved per thread: 4 for n <= 128 (product tables), 2 for larger
// trees, whose codes / tables / spill levels take more shared memory
static int prune_si(int n, int precision) {
    if (!wide_sites(n)) return 2;
    return precision == 32 ? PRUNE_SI32 : PRUNE_SI64;
}
int prune_batch_sites(int n, int precision) { return PRUNE_THREADS * prune_si(n, precision); }

// exact-sum units (arith.cuh Exact128): one log per thread per unit; 4-batch units on
// long alignments (the tiling is coarse there anyway), single batches below
// MPCGS_UNIT_MIN_BATCHES batches.  A function of the alignment only (P22).
#ifndef MPCGS_UNIT_MIN_BATCHES
#define MPCGS_UNIT_MIN_BATCHES 32
#endif
int prune_unit_batches(int n, int L, int precision) {
    const int batch = prune_batch_sites(n, precision);
    const long batches = (L + batch - 1) / batch;
    return batches >= MPCGS_UNIT_MIN_BATCHES ? 4 : 1;
}

// register need the table kernel serves (DR registers + PRUNE_SPILL shared levels);
// deeper trees (rare) are scored by the flat kernel in a second pass
// One shared spill level up to n = 64 (a random coalescent tree of 64 tips needs
// more than DR + 1 = 4 registers about once in 140), two above.
#ifndef MPCGS_SPILL64
#define MPCGS_SPILL64 1
#endif
int prune_need_cap(int n) { return std::min(prune_max_need(n), PRUNE_DR + (n <= 64 ? MPCGS_SPILL64 : PRUNE_SPILL)); }


template <typename T, bool GM>
static size_t tab_bytes_for(int n, bool amb = false, int bufs = 2) {
    const int cap = prune_need_cap(n);
    constexpr int SI = sizeof(T) == 4 ? PRUNE_SI32 : PRUNE_SI64;
    if (amb)  // 4-bit base-set codes, 16-row tip tables (S24)
        return wide_sites(n) ? tab_smem_bytes<T, PRUNE_DR, SI, false, GM, 4>(n - 1, cap, 0, bufs)
                             : tab_smem_bytes<T, PRUNE_DR, PRUNE_SI_LARGE, false, GM, 4>(n - 1, cap, 0, bufs);
    const bool pt = product_tables<T, GM>(n);
    if (pt && !wide_sites(n)) return tab_smem_bytes<T, PRUNE_DR, PRUNE_SI_LARGE, true, GM>(n - 1, cap, 0, bufs);
    return pt ? tab_smem_bytes<T, PRUNE_DR, SI, true, GM>(n - 1, cap, 0, bufs)
              : tab_smem_bytes<T, PRUNE_DR, PRUNE_SI_LARGE, false, GM>(n - 1, cap, 0, bufs);
}

// resident CTAs per SM the shared memory of `bytes` allows (228 KB per SM, 1 KB reserved per CTA)
static int by_smem(size_t bytes) { return (int)((228 * 1024) / (bytes + 1024 + 256)); }

// the layout launch_tab_w picks: one code buffer when that buys a resident CTA
template <typename T, bool GM>
static size_t tab_bytes_best(int n, bool amb = false) {
    const int regcap = sizeof(T) == 4 ? 4 : 3;
    const size_t b2 = tab_bytes_for<T, GM>(n, amb, 2), b1 = tab_bytes_for<T, GM>(n, amb, 1);
    return (MPCGS_SINGLEBUF && std::min(regcap, by_smem(b1)) > std::min(regcap, by_smem(b2))) ? b1 : b2;
}

#ifndef MPCGS_TAB_MIN_N
#define MPCGS_TAB_MIN_N 8  // below 8 tips the table setup costs more than it saves (c1: 41 -> 37 us per step)
#endif
// resident table-kernel CTAs per SM for the tiling cost model: the register limit
// (159 registers FP64 -> 3, FP32 -> 4) or the shared-memory limit of the base layout
int prune_resident_per_sm(int n, int precision, bool general_model) {
    size_t bytes;
    if (precision == 32) bytes = general_model ? tab_bytes_best<float, true>(n) : tab_bytes_best<float, false>(n);
    else bytes = general_model ? tab_bytes_best<double, true>(n) : tab_bytes_best<double, false>(n);
    return std::max(1, std::min(precision == 32 ? 4 : 3, by_smem(bytes)));
}

bool prune_uses_tables(int n, int precision, bool general_model, bool amb) {
    if (n < MPCGS_TAB_MIN_N) return false;
    size_t bytes;
    if (precision == 32) bytes = general_model ? tab_bytes_best<float, true>(n, amb) : tab_bytes_best<float, false>(n, amb);
    else bytes = general_model ? tab_bytes_best<double, true>(n, amb) : tab_bytes_best<double, false>(n, amb);
    return bytes <= 160 * 1024;
}

cudaError_t launch_prune(const PruneArgs& a, int ntrees, int depth, int precision, cudaStream_t st,
                         int* n_launched) {
    int nl = 0;
    cudaError_t e = cudaSuccess;
    if (ntrees > 0)
        e = precision == 32 ? (a.gm ? launch_prune_typed<float, true>(a, ntrees, depth, st, nl)
                                    : launch_prune_typed<float, false>(a, ntrees, depth, st, nl))
                            : (a.gm ? launch_prune_typed<double, true>(a, ntrees, depth, st, nl)
                                    : launch_prune_typed<double, false>(a, ntrees, depth, st, nl));
    if (n_launched) *n_launched = nl;
    return e;
}

}  // namespace mpcgs

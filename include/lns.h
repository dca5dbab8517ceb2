/*
 * lns.h -- C ABI of the B200 (sm_100a) large-neighbourhood tabu search for the Permuted
 * Perceptron Problem (Luong, Melab, Talbi, "Large Neighborhood Local Search Optimization on
 * Graphics Processing Units", LSPP @ IPDPS 2010; text in PAPER.md, cited as PAPER.md:<line>).
 *
 * The hot path: full evaluation of the k-Hamming neighbourhood (k = 1, 2, 3;
 * sizes n, C(n,2), C(n,3)) of the current +-1 solution V, selection of the
 * best non-tabu neighbour, and the move, inside a tabu search. Variant
 * k = 4..7 (the same method, generic-k kernel; see the note above lns_tabu_run).
 *
 * Conventions shared by every entry point
 *  - Problem (Definition 1): A is an m x n matrix with entries +-1, stored
 *    ROW-MAJOR as int8 (A[j*n + i]); S is the multiset of m non-negative ints (int32); V is a
 *    length-n int8 vector of +-1; Y = A V (int32, length m).
 *  - Fitness: f(V) = 30 * sum_j (|Y_j| - Y_j) + sum_{b=0..n} |H_b - H'_b|,
 *    H_b = #{j : S_j = b}, H'_b = #{j : Y_j = b}; bins 0..n (reading R1).
 *  - Neighbour ranks: a neighbour flips the k distinct bits i1 < i2 < i3; its rank is its index
 *    in LEXICOGRAPHIC order of (i1, i2, i3) (reading R6; the order of Prop. 1 / Appendix A for
 *    k = 2, and of the "set of plans" of Appendix C for k = 3).
 *  - Selection: the admissible neighbour of least fitness, ties to the LOWEST rank (R5); no
 *    aspiration (R4). Tabu list: FIFO of the last `tenure` accepted ranks (R3); default tenure
 *    floor(C(n,k)/6) ("m/6, m = number of neighbours").
 *  - Pointers marked (host|device) may point to host memory or to device memory of the
 *    context's device; the library detects which with cudaPointerGetAttributes. The caller
 *    owns every buffer it passes; the library copies what it keeps.
 *  - `stream` is a cudaStream_t (NULL = legacy default stream). Entry points that return
 *    results to the host synchronise that stream before returning.
 *  - Errors: every call returns an lns_status; the library never aborts. Asynchronous CUDA
 *    errors surface at the next synchronisation as LNS_ECUDA. lns_strerror() names a code;
 *    lns_last_error() gives a message for the last failure on the calling thread.
 *  - Limits: 1 <= n, 1 <= m; C(n,k) < 2^32 - 1 (n <= 2954 for k = 3); 60 m n + 2 m < 2^31
 *    (so fitness fits int32 and the (fitness, rank) key fits 63 bits); the bit-packed A of
 *    ceil(m/32) * n words must fit in shared memory (m*n <= ~1.3e6, e.g. 1024 x 1024).
 */
#ifndef LNS_H
#define LNS_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef int32_t lns_status;
#define LNS_OK 0
#define LNS_EINVAL (-1)         /* bad argument (k not in 1..7 or the call not available for k, n < k, A not +-1, S outside [0,n], Y != A V, ...) */
#define LNS_ERANGE (-2)         /* size limit exceeded (see Limits), or tenure >= C(n,k) */
#define LNS_ENOMEM (-3)         /* device or host allocation failed */
#define LNS_ECUDA (-4)          /* CUDA runtime error (message in lns_last_error) */
#define LNS_ENCCL (-5)          /* NCCL missing or failed */
#define LNS_ENOADMISSIBLE (-6)  /* every neighbour is tabu (best_rank = -1) */
#define LNS_EPEER (-7)          /* device-side peer exchange: a partition did not arrive in time */

#define LNS_IPC_HANDLE_BYTES 64 /* size of a cudaIpcMemHandle_t (lns_exchange_ipc_handle) */
#define LNS_UNIQUE_ID_BYTES 128 /* size of an ncclUniqueId (lns_get_unique_id) */

#define LNS_STOP_ON_ZERO 1      /* stop the search when f = 0 */
#define LNS_FORCE_STEPPED 2     /* run one launch sequence per iteration instead of the persistent kernel */
#define LNS_ASPIRATION 4        /* variant (not the default, reading R4'): a tabu move is admissible when its
                                   fitness is below the best fitness found so far (Taillard [11]) */
#define LNS_TABU_SOLUTIONS 16   /* variant (not the default, reading R3'): the tabu list holds the `tenure`
                                   most recently visited SOLUTIONS V_{t-L} .. V_{t-1} (PAPER.md:243-244 read
                                   literally), not move ranks; a neighbour is tabu iff it equals one of
                                   them. lns_tabu_run (persistent kernel, also with peers) and
                                   lns_tabu_run_batch only; tenure >= 1. The visited ring costs tenure x
                                   ceil(n/32) x 4 bytes of device memory per concurrent search. */
#define LNS_PLAIN_LAUNCH 8      /* lns_tabu_run: launch the persistent kernel with a plain launch instead of
                                   a cooperative one. The driver serialises cooperative launches, so several
                                   peer partitions on ONE device (tests, emulation) need this; co-residency
                                   is then not guaranteed (an idle device with room for all CTAs gives it;
                                   the peer exchange times out otherwise). */

typedef struct lns_ctx lns_ctx;

/* Outcome of one tabu search (PAPER.md:256-258 report fitness, #iterations and success). */
typedef struct {
    int64_t iters_done;      /* iterations performed (an iteration = evaluate all C(n,k) + move) */
    int64_t final_f;         /* fitness of the final solution */
    int64_t best_f;          /* least fitness seen, including the start vector */
    int64_t best_iter;       /* first iteration reaching best_f (0 = start vector) */
    int64_t first_zero_iter; /* first iteration with f = 0 (0 = start, -1 = never) */
    int32_t solved;          /* best_f == 0 */
    int32_t reserved;
} lns_result;

/* lns_create -- upload one PPP instance (Definition 1) to `device`.
 *   A: (host|device) m x n int8 row-major, entries +-1.  S: (host|device) m int32 in [0, n].
 *   The library bit-packs A and builds the histogram H of S; the caller
 *   keeps A and S. *out receives a context owned by the library until lns_destroy.
 *   Errors: EINVAL (m < 1, n < 1, entry of A not +-1, S_j outside [0,n]), ERANGE (limits),
 *   ENOMEM, ECUDA. */
lns_status lns_create(const int8_t *A, int32_t m, int32_t n, const int32_t *S, int32_t device,
                      lns_ctx **out);

/* lns_destroy -- free everything the context owns (NULL is a no-op). */
void lns_destroy(lns_ctx *ctx);

/* lns_eval_neighborhood -- evaluate all C(n,k) neighbours of V (Figs. 7/9/10, PAPER.md:212-216,
 *   371-383, 405-413) and return the admissible neighbour of least fitness, lowest rank on ties.
 *   V: (host|device) n int8 +-1.  Y: (host|device) m int32, must equal A V (verified on the
 *   device; EINVAL otherwise).  tabu_bits: (host|device) ceil(C(n,k)/32) uint32 words,
 *   bit r%32 of word r/32 set <=> rank r is tabu; NULL = nothing tabu.  If a partition was set
 *   (lns_set_partition / lns_attach_comm) only that slice of ranks is evaluated.
 *   best_fitness, best_rank: host int64 outputs. Synchronous.
 *   Errors: EINVAL, ERANGE, ENOADMISSIBLE (all evaluated ranks tabu: best_rank = -1,
 *   best_fitness = -1), ECUDA. */
lns_status lns_eval_neighborhood(lns_ctx *ctx, int32_t k, const int8_t *V, const int32_t *Y,
                                 const uint32_t *tabu_bits, int64_t *best_fitness,
                                 int64_t *best_rank, void *stream);

/* lns_eval_all -- the fitness of every neighbour of V, by rank (the paper's new_fitness[]
 *   array).  fitness_out: (host|device) C(n,k) int32.  Ignores partitions.
 *   Synchronous. Errors: EINVAL, ERANGE, ECUDA. */
lns_status lns_eval_all(lns_ctx *ctx, int32_t k, const int8_t *V, int32_t *fitness_out, void *stream);

/* lns_tabu_run -- tabu search of PAPER.md:241-258: `iters` iterations (or until f = 0 when
 *   flags & LNS_STOP_ON_ZERO), each evaluating every neighbour and moving to the best
 *   admissible one (tie -> lowest rank), with a FIFO tabu list of `tenure` ranks
 *   (tenure < 0 -> floor(C(n,k)/6)).
 *   V0: (host|device) n int8 +-1, or NULL -> drawn from `seed` (splitmix64, reading R12:
 *   ceil(n/64) draws, bit i LSB-first, 1 -> -1).
 *   V_out: (host|device) n int8 final solution, nullable.  trace_rank, trace_fit:
 *   (host|device) int64 arrays of length `iters`, nullable; entry t-1 = (rank, fitness) accepted
 *   at iteration t.  res: host, required.  With a communicator attached (lns_attach_comm) every
 *   rank of the communicator must call this with identical arguments: each GPU evaluates its
 *   slice of ranks and one NCCL u64-MIN all-reduce per iteration picks the global move; the
 *   trajectory is identical for any number of GPUs.  Synchronous.
 *   Errors: EINVAL, ERANGE (limits, tenure >= C(n,k)), ENOMEM, ECUDA, ENCCL. */
/* k > 3 (PAPER.md:105-125 generalised; 4 <= k <= 7): lns_tabu_run (one
 *   device, persistent kernel, rank tabu list with or without LNS_ASPIRATION),
 *   lns_tabu_run_batch (the same per restart), lns_eval_neighborhood (no partition),
 *   lns_eval_all and lns_unrank only; m <= 255 (the byte window) else ERANGE; other calls and
 *   flags with k > 3 return EINVAL. */
lns_status lns_tabu_run(lns_ctx *ctx, int32_t k, int64_t iters, int64_t tenure, uint64_t seed,
                        const int8_t *V0, int32_t flags, int8_t *V_out, int64_t *trace_rank,
                        int64_t *trace_fit, lns_result *res, void *stream);

/* lns_tabu_run_batch -- R independent searches (restarts) of lns_tabu_run (the paper runs every
 *   configuration 50 times).
 *   Restart r starts from V0 + r*n when V0 != NULL, else from the splitmix64 vector of
 *   seed_r = first splitmix64 output of a stream seeded with seed + r (reading R12).
 *   V_out: (host|device) R x n int8, nullable.  res: host, R entries.  Partitions set with
 *   lns_set_partition are ignored (each restart runs whole on one device). With a communicator
 *   attached (lns_attach_comm / lns_comm_init_rank, world G > 1) every rank must call this with
 *   identical arguments: restart r runs on rank r mod G, and every rank receives all R results
 *   and final vectors (gathered by NCCL sums of zero-padded arrays; no per-iteration
 *   collective).  Synchronous.
 *   Errors: as lns_tabu_run. */
lns_status lns_tabu_run_batch(lns_ctx *ctx, int32_t k, int32_t R, int64_t iters, int64_t tenure,
                              uint64_t seed, const int8_t *V0, int32_t flags, int8_t *V_out,
                              lns_result *res, void *stream);

/* lns_unrank -- flip sets of ranks (device kernel; used by tests of the rank order).
 *   k = 4..7: out is count x k int32 (the generic-k unranking of the k > 3 kernel).
 *   ranks: (host|device) count int64 in [0, C(n,k)).  out: (host|device) count x 3 int32,
 *   unused slots -1.  Synchronous. Errors: EINVAL (rank out of range), ERANGE, ECUDA. */
lns_status lns_unrank(int32_t n, int32_t k, const int64_t *ranks, int64_t count, int32_t *out,
                      void *stream);

/* lns_set_partition -- restrict evaluation to slice `part` of `nparts` of the rank space
 *   ("partitioning the neighborhood set, where each partition is executed on
 *   a single GPU"). Slice g = [B(g), B(g+1)), B(g) = 32 * floor(C(n,k) * g / (32 nparts)),
 *   B(nparts) = C(n,k). Errors: EINVAL. */
lns_status lns_set_partition(lns_ctx *ctx, int32_t part, int32_t nparts);

/* lns_attach_comm -- borrow an NCCL communicator (ncclComm_t) for multi-GPU lns_tabu_run /
 *   lns_tabu_run_batch; sets the partition to (rank, world). The communicator
 *   must come from the libnccl ALREADY LOADED in the process (e.g. torch's, via
 *   ProcessGroupNCCL._comm_ptr()): ncclAllReduce is looked up in that copy only (dlopen
 *   RTLD_NOLOAD of libnccl.so.2, else the global symbol scope), never in a freshly loaded one.
 *   The communicator is borrowed (not freed). comm = NULL detaches (and destroys a communicator
 *   made by lns_comm_init_rank).
 *   Errors: EINVAL (rank/world), ENCCL (no libnccl loaded in the process). */
lns_status lns_attach_comm(lns_ctx *ctx, void *nccl_comm, int32_t rank, int32_t world);

/* NCCL bootstrap without torch (one process per GPU, plain C callers):
 *   lns_get_unique_id  -- on ONE rank: write a fresh ncclUniqueId (LNS_UNIQUE_ID_BYTES bytes,
 *                         host buffer) to id_out; the caller distributes it to every rank
 *                         (MPI, a file, a socket...).
 *   lns_comm_init_rank -- on EVERY rank (collective over `world` processes): create an NCCL
 *                         communicator from that id on the context's device (ncclCommInitRank),
 *                         owned by the context, and attach it as lns_attach_comm would (partition
 *                         (rank, world)). Destroyed by lns_destroy or lns_attach_comm(NULL).
 *   Both use the libnccl already loaded in the process, else load libnccl.so.2 (the same copy
 *   then serves every call on that communicator).
 *   Errors: EINVAL (null id, rank/world), ENCCL (libnccl not found, NCCL call failed). */
lns_status lns_get_unique_id(uint8_t *id_out);
lns_status lns_comm_init_rank(lns_ctx *ctx, const uint8_t *id, int32_t rank, int32_t world);

/* Device-initiated multi-GPU exchange (the partition of P:448-454 with
 * the per-iteration argmin moved inside the persistent kernel, no host collective):
 *   Every partition's kernel owns a 512-byte exchange buffer in its device memory. At iteration t
 *   every CTA of every partition MINs its best key into slot t mod 3 of EVERY partition's buffer
 *   (red.min.sys over NVLink peer memory) and then bumps every partition's arrival counter
 *   (red.release.sys); it proceeds once its own counter shows all CTAs of all partitions
 *   (ld.acquire.sys), reads its own slot (the global minimum) and applies the move. A partition
 *   that does not arrive within timeout_ms ends the run with LNS_EPEER (no hang).
 *   lns_exchange_buffer      -- this context's exchange buffer (device pointer; allocated here).
 *   lns_exchange_ipc_handle  -- its cudaIpcMemHandle_t (LNS_IPC_HANDLE_BYTES, host) for other
 *                               processes (one process per GPU).
 *   lns_attach_peers         -- set the partition (part of nparts) and the exchange buffers of all
 *                               partitions, bufs[q] a device pointer usable from this context's
 *                               device (bufs[part] = this context's own buffer; peers on other
 *                               GPUs need peer access enabled). nparts = 1 or bufs = NULL detaches.
 *   lns_attach_peers_ipc     -- the same from nparts handles (host, nparts x LNS_IPC_HANDLE_BYTES,
 *                               gathered from every partition); opens the other partitions'
 *                               buffers with cudaIpcOpenMemHandle (closed by lns_destroy).
 *   lns_exchange_reset       -- clear this context's own buffer and wait for it. Before EVERY
 *                               lns_tabu_run with peers attached, every partition must reset its
 *                               buffer and pass a host barrier, then all call lns_tabu_run with
 *                               identical arguments (each evaluates its slice; the trajectory is
 *                               the single-GPU one). Only lns_tabu_run uses the peers.
 *   Errors: EINVAL (bad partition / pointers), ENOMEM, ECUDA (IPC); lns_tabu_run: EPEER. */
lns_status lns_exchange_buffer(lns_ctx *ctx, void **buf_dev);
lns_status lns_exchange_ipc_handle(lns_ctx *ctx, void *handle_out);
lns_status lns_attach_peers(lns_ctx *ctx, int32_t part, int32_t nparts, void *const *bufs,
                            int64_t timeout_ms);
lns_status lns_attach_peers_ipc(lns_ctx *ctx, int32_t part, int32_t nparts, const void *handles,
                                int64_t timeout_ms);
lns_status lns_exchange_reset(lns_ctx *ctx, void *stream);

/* Stepped interface (one iteration at a time; used by multi-process drivers that own the
 * collective, e.g. torch.distributed):
 *   lns_step_begin  -- start a search (arguments as lns_tabu_run; trace capacity = max_iters).
 *   lns_step_eval   -- evaluate this context's slice for the current iteration and store the
 *                      partial best key ((fitness << 32) | rank, or INT64_MAX if nothing is
 *                      admissible) into key_dev[0] (device int64). Asynchronous on `stream`.
 *   lns_step_apply  -- key_dev[0] now holds the GLOBAL minimum key (after an all-reduce MIN):
 *                      apply that move, update the tabu list and the trace. Asynchronous.
 *   lns_step_end    -- copy out V_out / traces / result as lns_tabu_run does. Synchronous.
 * Iterations after f = 0 (with LNS_STOP_ON_ZERO) are no-ops on the device. */
lns_status lns_step_begin(lns_ctx *ctx, int32_t k, int64_t max_iters, int64_t tenure, uint64_t seed,
                          const int8_t *V0, int32_t flags, void *stream);
lns_status lns_step_eval(lns_ctx *ctx, int64_t *key_dev, void *stream);
lns_status lns_step_apply(lns_ctx *ctx, const int64_t *key_dev, void *stream);
lns_status lns_step_end(lns_ctx *ctx, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit,
                        lns_result *res, void *stream);

/* lns_last_kernel_ms -- device time (CUDA events) of the hot kernel(s) of the last run or eval. */
double lns_last_kernel_ms(lns_ctx *ctx);

/* lns_config -- override launch parameters (0 = automatic): CTAs per search (lns_tabu_run,
 * the stepped API) and CTAs of lns_eval_all / lns_eval_neighborhood. Results never depend on it. */
lns_status lns_config(lns_ctx *ctx, int32_t blocks);

int64_t lns_neighborhood_size(int32_t n, int32_t k); /* C(n,k), or -1 if k not in 1..7 */
const char *lns_strerror(lns_status status);
const char *lns_last_error(void);
int32_t lns_version(void); /* major*10000 + minor*100 + patch */

/* Device-memory cache of the library (a runtime component, not a passage of the paper).
 * Context buffers (lns_create, the per-run until[] / trace / restart arrays) come from a per-device
 * caching allocator: lns_destroy returns them to a cache keyed by (device, power-of-two size
 * class) instead of cudaFree, so create -> run -> destroy cycles do not pay cudaMalloc / cudaFree
 * (which synchronises the device). The cache holds at most LNS_POOL_CAP_MB (environment, read once,
 * default 4096) MiB; beyond that blocks are freed. An allocation that fails retries once after
 * releasing the cache.
 * lns_pool_trim -- cudaFree every cached (unused) block on every device. Thread-safe; never fails.
 * lns_pool_stats -- bytes currently cached (unused) and handed out (in use by live contexts);
 *                   either pointer may be NULL. */
void lns_pool_trim(void);
void lns_pool_stats(int64_t *cached_bytes, int64_t *live_bytes);

/* ---------------------------------------------------------------------------------------------
 * Second binary fitness: UBQP (SURVEY.md §8(f) f4 "a pluggable binary fitness").
 * The paper states its neighbourhood mappings "for binary problems" and
 * validates them on the PPP only. Here the same k-Hamming tabu search (neighbourhood
 * PAPER.md:105-125, lexicographic ranks R6, until[] tabu list R3 with default tenure
 * floor(C(n,k)/6), least fitness / lowest rank R5, no aspiration R4) minimises
 *     f(x) = x^T Q x = sum_i sum_j Q_ij x_i x_j,   x in {0,1}^n,  Q symmetric int32.
 * k in {1, 2, 3}. Vectors are uint8 0/1 (NOT the +-1 int8 of the PPP calls).
 * ------------------------------------------------------------------------------------------- */
typedef struct lns_bqp lns_bqp;

/* lns_bqp_create -- upload Q ((host|device) n x n int32 row-major, symmetric) to `device`; the
 *   caller keeps Q. *out receives a context owned by the library until lns_bqp_destroy.
 *   Errors: EINVAL (n < 1, Q not symmetric, bad device), ERANGE (n > 4096, or sum |Q_ij| >= 2^29:
 *   the kernels compute fitnesses exactly in int32), ENOMEM, ECUDA. */
lns_status lns_bqp_create(const int32_t *Q, int32_t n, int32_t device, lns_bqp **out);

/* lns_bqp_destroy -- free everything the context owns (NULL is a no-op). */
void lns_bqp_destroy(lns_bqp *ctx);

/* lns_bqp_eval_all -- f(x xor F_r) of every neighbour r of x, by lexicographic rank.
 *   x: (host|device) n uint8 0/1.  fitness_out: (host|device) C(n,k) int32.  Synchronous
 *   (ordered after `stream`). Errors: EINVAL (k not 1..3, n < k, x not 0/1), ERANGE
 *   (C(n,k) >= 2^32 - 1), ENOMEM, ECUDA. */
lns_status lns_bqp_eval_all(lns_bqp *ctx, int32_t k, const uint8_t *x, int32_t *fitness_out, void *stream);

/* lns_bqp_tabu_run -- `iters` iterations of the tabu search from x0 ((host|device) n uint8 0/1),
 *   tenure < 0 -> floor(C(n,k)/6). Outputs (each may be NULL except res; host or device):
 *   x_out n uint8, trace_rank / trace_fit `iters` int64 (accepted rank and fitness per
 *   iteration), res[4] (host) = {iterations done, final f, best f, first iteration reaching best
 *   f (0 = x0)}. Synchronous (ordered after `stream`; the library runs on a private stream
 *   and replays the per-iteration eval + apply launches from a CUDA graph).
 *   Errors: EINVAL, ERANGE (tenure >= C(n,k), iters + tenure >= 2^32), ENOMEM, ECUDA. */
lns_status lns_bqp_tabu_run(lns_bqp *ctx, int32_t k, int64_t iters, int64_t tenure, const uint8_t *x0,
                            uint8_t *x_out, int64_t *trace_rank, int64_t *trace_fit, int64_t *res,
                            void *stream);

/* lns_bqp_tabu_run_batch -- R independent searches of `iters` iterations each, run side by side
 *   (restart r from x0s + r n; the paper's protocol runs every configuration 50 times, PAPER.md:
 *   249-252): every iteration evaluates all R neighbourhoods in one launch (grid row r = restart r)
 *   and applies the R moves in one launch, replayed from a CUDA graph. Each restart follows exactly
 *   the trajectory lns_bqp_tabu_run gives from the same start. x0s: (host|device) R x n uint8 0/1;
 *   x_outs: nullable (host|device) R x n uint8; res (host) R x 4 int64, row r as res of
 *   lns_bqp_tabu_run. R in [1, 65535]; device memory R x C(n,k) x 4 bytes for the tabu lists.
 *   Synchronous (ordered after `stream`). Errors: as lns_bqp_tabu_run; EINVAL also for R < 1,
 *   ERANGE for R > 65535, ENOMEM when the R tabu lists do not fit. */
lns_status lns_bqp_tabu_run_batch(lns_bqp *ctx, int32_t k, int32_t R, int64_t iters, int64_t tenure,
                                  const uint8_t *x0s, uint8_t *x_outs, int64_t *res, void *stream);

/* lns_bqp_last_kernel_ms -- device time (CUDA events) of the last eval_all / tabu_run (-1: NULL). */
double lns_bqp_last_kernel_ms(const lns_bqp *ctx);

#ifdef __cplusplus
}
#endif
#endif /* LNS_H */

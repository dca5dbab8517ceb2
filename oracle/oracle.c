/*
 * oracle.c -- CPU ORACLE for the k-Hamming tabu search on the Permuted Perceptron Problem
 * (Luong, Melab, Talbi, "Large Neighborhood Local Search Optimization on GPUs", LSPP@IPDPS 2010;
 * text in PAPER.md).
 *
 * THIS IS TEST INFRASTRUCTURE. Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load it. It shares no code with the CUDA path
 * (paper_conf_ipps_luongmt10_b200/csrc): no headers, helpers, tables or constants. The product
 * path never calls it.
 *
 * Style: plain and slow. Every fitness is recomputed FROM SCRATCH for every neighbour; the
 * neighbourhood is enumerated with nested loops whose loop counter IS the rank (no index
 * formula); the tabu list is the literal "until" array. The only "trick" is the textbook
 * identity <a, v> = n - 2 popcount(a xor v) for +-1 vectors stored as sign bits, used by the
 * *_packed variants for speed; the scalar variants do the int8 multiply-add and the tests check
 * that the two agree.
 *
 * Parity status: every function is pinned by tests/test_oracle.py:
 *   fitness      -- hand-computed golden values, f(V*) = 0 on planted instances, brute force
 *                   zero set == multiset equality, f >= 0, parity f = #negative rows (mod 2)
 *   rank order   -- itertools.combinations order (k = 1..7), the paper's worked example
 *                   (n = 6, (2,3) -> 9), Appendix A-D formulas, C(n,k) counts
 *   selection    -- brute-force argmin with lowest-rank tie-break, tabu invariants
 *   trajectory   -- stop-on-zero reaches a vector whose multiset equals S
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#ifdef _OPENMP
#include <omp.h>
#endif

/* ---------------------------------------------------------------------------------------
 * splitmix64 (reading R12 of DESIGN.md): one draw = s += 0x9E3779B97F4A7C15, then mix.
 * Used only to derive V0 from a seed, exactly as ppp_inputs.start_vector does.
 * ------------------------------------------------------------------------------------- */
uint64_t oracle_splitmix64_next(uint64_t *s)
{
    uint64_t z;
    *s += 0x9E3779B97F4A7C15ULL;
    z = *s;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ULL;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBULL;
    return z ^ (z >> 31);
}

/* V0 in {+1,-1}^n: ceil(n/64) draws, bit i of the stream (LSB first) = 1 -> -1. */
void oracle_start_vector(int32_t n, uint64_t seed, int8_t *V)
{
    uint64_t s = seed, w = 0;
    for (int32_t i = 0; i < n; i++) {
        if (i % 64 == 0) w = oracle_splitmix64_next(&s);
        V[i] = ((w >> (i % 64)) & 1) ? -1 : 1;
    }
}

/* ---------------------------------------------------------------------------------------
 * Histogram of Definition 1 / PAPER.md:227-229: H_b = #{ j : S_j = b }, b = 0..n.
 * (Reading R1: bins 0..n; reading R2: H is the histogram of the given multiset S.)
 * ------------------------------------------------------------------------------------- */
static void histogram_of(const int32_t *vals, int32_t m, int32_t n, int32_t *H)
{
    for (int32_t b = 0; b <= n; b++) H[b] = 0;
    for (int32_t j = 0; j < m; j++)
        if (vals[j] >= 0 && vals[j] <= n) H[vals[j]]++;
}

/* ---------------------------------------------------------------------------------------
 * Fitness, PAPER.md:231-237 (Section IV-A):
 *   f(V') = 30 * sum_{j=1..m} ( |(AV')_j| - (AV')_j ) + sum_{b} | H_b - H'_b |
 * with H' the histogram of Y' = AV' over bins b = 0..n (reading R1). Scalar int8 path.
 * ------------------------------------------------------------------------------------- */
static int64_t fitness_from_Y(const int32_t *Y, int32_t m, int32_t n, const int32_t *H, int32_t *Hp)
{
    int64_t pen = 0, hst = 0;
    histogram_of(Y, m, n, Hp);
    for (int32_t j = 0; j < m; j++) {
        int64_t y = Y[j];
        pen += (y < 0 ? -y : y) - y;
    }
    for (int32_t b = 0; b <= n; b++) {
        int64_t d = (int64_t)H[b] - Hp[b];
        hst += d < 0 ? -d : d;
    }
    return 30 * pen + hst;
}

int64_t oracle_fitness(const int8_t *A, int32_t m, int32_t n, const int32_t *S, const int8_t *V)
{
    int32_t *Y = malloc(sizeof(int32_t) * (size_t)m);
    int32_t *H = malloc(sizeof(int32_t) * (size_t)(n + 1));
    int32_t *Hp = malloc(sizeof(int32_t) * (size_t)(n + 1));
    histogram_of(S, m, n, H);
    for (int32_t j = 0; j < m; j++) { /* Y = A V' (Definition 1) */
        int32_t acc = 0;
        for (int32_t i = 0; i < n; i++) acc += (int32_t)A[(size_t)j * n + i] * V[i];
        Y[j] = acc;
    }
    int64_t f = fitness_from_Y(Y, m, n, H, Hp);
    free(Y); free(H); free(Hp);
    return f;
}

/* ---------------------------------------------------------------------------------------
 * Packed representation for speed: a +-1 vector is stored as sign bits (bit = 1 <=> -1), 64 per
 * word. Textbook identity: for x, v in {+-1}^n, <x, v> = n - 2 * popcount(bits(x) xor bits(v)).
 * ------------------------------------------------------------------------------------- */
typedef struct {
    int32_t m, n, nw;      /* nw = ceil(n/64) */
    uint64_t *abits;       /* m rows x nw words */
    int32_t *H;            /* n+1 bins of S */
} packed_t;

static void pack_instance(const int8_t *A, int32_t m, int32_t n, const int32_t *S, packed_t *P)
{
    P->m = m; P->n = n; P->nw = (n + 63) / 64;
    P->abits = calloc((size_t)m * P->nw, sizeof(uint64_t));
    P->H = malloc(sizeof(int32_t) * (size_t)(n + 1));
    for (int32_t j = 0; j < m; j++)
        for (int32_t i = 0; i < n; i++)
            if (A[(size_t)j * n + i] < 0) P->abits[(size_t)j * P->nw + i / 64] |= 1ULL << (i % 64);
    histogram_of(S, m, n, P->H);
}

static void free_packed(packed_t *P) { free(P->abits); free(P->H); }

static void pack_vector(const int8_t *V, int32_t n, uint64_t *vb)
{
    int32_t nw = (n + 63) / 64;
    for (int32_t w = 0; w < nw; w++) vb[w] = 0;
    for (int32_t i = 0; i < n; i++)
        if (V[i] < 0) vb[i / 64] |= 1ULL << (i % 64);
}

/* From-scratch fitness of the packed vector vb (scratch buffers Y, Hp of sizes m, n+1). */
static int64_t fitness_packed(const packed_t *P, const uint64_t *vb, int32_t *Y, int32_t *Hp)
{
    for (int32_t j = 0; j < P->m; j++) {
        int32_t d = 0;
        const uint64_t *a = P->abits + (size_t)j * P->nw;
        for (int32_t w = 0; w < P->nw; w++) d += __builtin_popcountll(a[w] ^ vb[w]);
        Y[j] = P->n - 2 * d;
    }
    return fitness_from_Y(Y, P->m, P->n, P->H, Hp);
}

int64_t oracle_fitness_packed(const int8_t *A, int32_t m, int32_t n, const int32_t *S, const int8_t *V)
{
    packed_t P;
    pack_instance(A, m, n, S, &P);
    uint64_t *vb = malloc(sizeof(uint64_t) * (size_t)P.nw);
    int32_t *Y = malloc(sizeof(int32_t) * (size_t)m);
    int32_t *Hp = malloc(sizeof(int32_t) * (size_t)(n + 1));
    pack_vector(V, n, vb);
    int64_t f = fitness_packed(&P, vb, Y, Hp);
    free(vb); free(Y); free(Hp); free_packed(&P);
    return f;
}

/* ---------------------------------------------------------------------------------------
 * Neighbourhoods, PAPER.md:105-125 (Section II): flip 1, 2 or 3 bits. The neighbourhood
 * index space is enumerated by NESTED LOOPS i1 < i2 < i3 in increasing order; the rank of a
 * flip set is the loop counter (reading R6: lexicographic order, the order of Prop. 1 /
 * Appendix A for k = 2 and of the "set of plans" of Appendix C for k = 3).
 * first_count[i1] = number of flip sets whose smallest index is i1, counted by a loop.
 * ------------------------------------------------------------------------------------- */
#define ORACLE_KMAX 7

/* k >= 4 ("k > 3 via the combinatorial number system"): the flip sets are
 * still enumerated in lexicographic order by nested loops -- an odometer over i1 < i2 < ... < ik
 * (the innermost index runs fastest; when it cannot advance, the next one out advances and the
 * inner ones restart right after it) -- and the rank is still the loop counter. The number of
 * flip sets whose smallest index is i1 is the number of (k-1)-subsets of {i1+1, ..., n-1},
 * counted with Pascal's rule (subsets of a set of a elements: C(a, r) = C(a-1, r-1) + C(a-1, r)). */
static int64_t subsets(int32_t a, int32_t r)
{
    int64_t row[ORACLE_KMAX + 1];
    if (r < 0 || r > a) return 0;
    for (int32_t j = 0; j <= r; j++) row[j] = (j == 0);
    for (int32_t x = 1; x <= a; x++)
        for (int32_t j = (x < r ? x : r); j >= 1; j--) row[j] += row[j - 1];
    return row[r];
}

/* First flip set after idx[0..k-1] in lexicographic order, keeping idx[0..fixed-1]: 0 at the end. */
static int odometer_next(int32_t *idx, int32_t k, int32_t n, int32_t fixed)
{
    int32_t j = k - 1;
    while (j >= fixed && idx[j] == n - k + j) j--;
    if (j < fixed) return 0;
    idx[j]++;
    for (int32_t q = j + 1; q < k; q++) idx[q] = idx[q - 1] + 1;
    return 1;
}

static int64_t count_with_first(int32_t n, int32_t k, int32_t i1)
{
    int64_t c = 0;
    if (k >= 4) return subsets(n - 1 - i1, k - 1);
    if (k == 1) return 1;
    for (int32_t i2 = i1 + 1; i2 < n; i2++) {
        if (k == 2) c += 1;
        else c += n - 1 - i2; /* the i3 loop runs over i2+1 .. n-1 */
    }
    return c;
}

/* Number of neighbours C(n,k), counted by the same loops. */
int64_t oracle_neighborhood_size(int32_t n, int32_t k)
{
    int64_t c = 0;
    for (int32_t i1 = 0; i1 < n; i1++) c += count_with_first(n, k, i1);
    return c;
}

/* Flip sets of the given ranks (ascending), by walking the nested loops once. */
int32_t oracle_flipsets(int32_t n, int32_t k, const int64_t *ranks, int64_t cnt, int32_t *out)
{
    int64_t r = 0, q = 0;
    if (k >= 4 && k <= ORACLE_KMAX && k <= n) { /* the odometer; rows of k indices */
        int32_t idx[ORACLE_KMAX];
        for (int32_t j = 0; j < k; j++) idx[j] = j;
        do {
            while (q < cnt && ranks[q] == r) {
                for (int32_t j = 0; j < k; j++) out[(int64_t)k * q + j] = idx[j];
                q++;
            }
            r++;
        } while (q < cnt && odometer_next(idx, k, n, 0));
        return q == cnt ? 0 : -1;
    }
    if (k < 1 || k > 3) return -1;
    for (int32_t i1 = 0; i1 < n && q < cnt; i1++) {
        int32_t i2s = (k >= 2) ? i1 + 1 : 0, i2e = (k >= 2) ? n : 1;
        for (int32_t i2 = i2s; i2 < i2e && q < cnt; i2++) {
            int32_t i3s = (k == 3) ? i2 + 1 : 0, i3e = (k == 3) ? n : 1;
            for (int32_t i3 = i3s; i3 < i3e && q < cnt; i3++, r++) {
                while (q < cnt && ranks[q] == r) {
                    out[3 * q] = i1;
                    out[3 * q + 1] = (k >= 2) ? i2 : -1;
                    out[3 * q + 2] = (k == 3) ? i3 : -1;
                    q++;
                }
            }
        }
    }
    return q == cnt ? 0 : -1;
}

/* ---------------------------------------------------------------------------------------
 * Evaluate every neighbour of V (Figs. 7/9/10: new_fitness[move_index] = compute_fitness(V, move))
 * from scratch. mode 0: write all fitnesses to f_all (length C(n,k)); mode 1: only return
 * the best admissible (f, r), admissible(r) <=> until[r] < t (reading R3), lowest rank wins
 * ties (reading R5). `sample` (sorted ranks, mode 2) evaluates only those ranks into f_all.
 * ------------------------------------------------------------------------------------- */
typedef struct { int64_t f, r; } fr_t;

static void flip(uint64_t *vb, int32_t i) { vb[i / 64] ^= 1ULL << (i % 64); }

/* ---------------------------------------------------------------------------------------
 * Solution list (variant R3', flag 2 of oracle_tabu_run): the tabu list of PAPER.md:243-244
 * read literally -- "the solutions visited in the recent past". A plain open-addressing hash set
 * of the listed solutions (bit vectors, compared word for word), rebuilt from the list every
 * iteration.
 * ------------------------------------------------------------------------------------- */
typedef struct {
    int32_t nw;              /* words per solution */
    int64_t cap;             /* table slots (power of two) */
    const uint64_t **slot;   /* pointer to a listed solution, or NULL */
} solset_t;

static uint64_t hash_words(const uint64_t *v, int32_t nw)
{
    uint64_t h = 0x9E3779B97F4A7C15ULL;
    for (int32_t i = 0; i < nw; i++) {
        h ^= v[i];
        h *= 0xBF58476D1CE4E5B9ULL;
        h ^= h >> 31;
    }
    return h;
}

static int solset_contains(const solset_t *S, const uint64_t *v)
{
    for (int64_t i = (int64_t)(hash_words(v, S->nw) & (uint64_t)(S->cap - 1));; i = (i + 1) & (S->cap - 1)) {
        if (!S->slot[i]) return 0;
        if (memcmp(S->slot[i], v, sizeof(uint64_t) * (size_t)S->nw) == 0) return 1;
    }
}

static void solset_insert(solset_t *S, const uint64_t *v)
{
    int64_t i = (int64_t)(hash_words(v, S->nw) & (uint64_t)(S->cap - 1));
    while (S->slot[i]) {
        if (memcmp(S->slot[i], v, sizeof(uint64_t) * (size_t)S->nw) == 0) return; /* already listed */
        i = (i + 1) & (S->cap - 1);
    }
    S->slot[i] = v;
}

static fr_t scan_neighbourhood(const packed_t *P, const uint64_t *vb0, int32_t k, int mode,
                               int64_t *f_all, const int32_t *until, int64_t t,
                               const int64_t *sample, int64_t nsample, int nthreads, int64_t aspire_below,
                               const solset_t *sols)
{
    int32_t n = P->n;
    int64_t *base = malloc(sizeof(int64_t) * (size_t)(n + 1));
    base[0] = 0;
    for (int32_t i1 = 0; i1 < n; i1++) base[i1 + 1] = base[i1] + count_with_first(n, k, i1);
    fr_t best = { INT64_MAX, -1 };
#ifdef _OPENMP
    if (nthreads > 0) omp_set_num_threads(nthreads);
#endif
#pragma omp parallel
    {
        fr_t mine = { INT64_MAX, -1 };
        uint64_t *vb = malloc(sizeof(uint64_t) * (size_t)P->nw);
        int32_t *Y = malloc(sizeof(int32_t) * (size_t)P->m);
        int32_t *Hp = malloc(sizeof(int32_t) * (size_t)(n + 1));
#pragma omp for schedule(dynamic, 1)
        for (int32_t i1 = 0; i1 < n; i1++) {
            int64_t r = base[i1];
            int64_t q = 0;
            if (mode == 2) { /* first sampled rank >= r */
                int64_t lo = 0, hi = nsample;
                while (lo < hi) { int64_t mid = (lo + hi) / 2; if (sample[mid] < r) lo = mid + 1; else hi = mid; }
                q = lo;
                if (q >= nsample || sample[q] >= base[i1 + 1]) continue;
            }
            if (k >= 4) { /* odometer over i2 < ... < ik, i1 fixed */
                int32_t idx[ORACLE_KMAX];
                idx[0] = i1;
                for (int32_t j = 1; j < k; j++) idx[j] = i1 + j;
                if (idx[k - 1] >= n) continue;
                do {
                    if (mode == 2 && (q >= nsample || sample[q] != r)) { r++; continue; }
                    int tabu = (mode == 1 && until && !(until[r] < t));
                    if (tabu && aspire_below < 0) { r++; continue; }
                    memcpy(vb, vb0, sizeof(uint64_t) * (size_t)P->nw);
                    for (int32_t j = 0; j < k; j++) flip(vb, idx[j]);
                    if (mode == 1 && sols && solset_contains(sols, vb)) {
                        tabu = 1;
                        if (aspire_below < 0) { r++; continue; }
                    }
                    int64_t f = fitness_packed(P, vb, Y, Hp);
                    if (!(tabu && !(f < aspire_below))) {
                        if (mode == 0) f_all[r] = f;
                        else if (mode == 2) { while (q < nsample && sample[q] == r) { f_all[q] = f; q++; } }
                        else if (f < mine.f || (f == mine.f && r < mine.r)) { mine.f = f; mine.r = r; }
                    }
                    r++;
                } while (odometer_next(idx, k, n, 1));
                continue;
            }
            int32_t i2s = (k >= 2) ? i1 + 1 : 0, i2e = (k >= 2) ? n : 1;
            for (int32_t i2 = i2s; i2 < i2e; i2++) {
                int32_t i3s = (k == 3) ? i2 + 1 : 0, i3e = (k == 3) ? n : 1;
                for (int32_t i3 = i3s; i3 < i3e; i3++, r++) {
                    if (mode == 2) {
                        if (q >= nsample || sample[q] != r) continue;
                    }
                    int tabu = (mode == 1 && until && !(until[r] < t));
                    if (tabu && aspire_below < 0) continue; /* tabu, no aspiration */
                    memcpy(vb, vb0, sizeof(uint64_t) * (size_t)P->nw);
                    flip(vb, i1);
                    if (k >= 2) flip(vb, i2);
                    if (k == 3) flip(vb, i3);
                    if (mode == 1 && sols && solset_contains(sols, vb)) { /* V' is a listed solution */
                        tabu = 1;
                        if (aspire_below < 0) continue;
                    }
                    int64_t f = fitness_packed(P, vb, Y, Hp);
                    /* aspiration (reading R4'): a tabu move is admissible if it beats the best
                     * fitness found so far */
                    if (tabu && !(f < aspire_below)) continue;
                    if (mode == 0) f_all[r] = f;
                    else if (mode == 2) { while (q < nsample && sample[q] == r) { f_all[q] = f; q++; } }
                    else if (f < mine.f || (f == mine.f && r < mine.r)) { mine.f = f; mine.r = r; }
                }
            }
        }
#pragma omp critical
        {
            if (mine.f < best.f || (mine.f == best.f && mine.r < best.r)) best = mine;
        }
        free(vb); free(Y); free(Hp);
    }
    free(base);
    return best;
}

int32_t oracle_eval_all(const int8_t *A, int32_t m, int32_t n, const int32_t *S, const int8_t *V,
                        int32_t k, int64_t *f_all, int32_t nthreads)
{
    if (k < 1 || k > ORACLE_KMAX || n < k) return -1;
    packed_t P;
    pack_instance(A, m, n, S, &P);
    uint64_t *vb = malloc(sizeof(uint64_t) * (size_t)P.nw);
    pack_vector(V, n, vb);
    scan_neighbourhood(&P, vb, k, 0, f_all, NULL, 0, NULL, 0, nthreads, -1, NULL);
    free(vb); free_packed(&P);
    return 0;
}

/* Fitness of sampled neighbours (ranks ascending) -- for full-size parity on sampled outputs. */
int32_t oracle_eval_ranks(const int8_t *A, int32_t m, int32_t n, const int32_t *S, const int8_t *V,
                          int32_t k, const int64_t *ranks, int64_t cnt, int64_t *f_out, int32_t nthreads)
{
    if (k < 1 || k > ORACLE_KMAX || n < k) return -1;
    packed_t P;
    pack_instance(A, m, n, S, &P);
    uint64_t *vb = malloc(sizeof(uint64_t) * (size_t)P.nw);
    pack_vector(V, n, vb);
    scan_neighbourhood(&P, vb, k, 2, f_out, NULL, 0, ranks, cnt, nthreads, -1, NULL);
    free(vb); free_packed(&P);
    return 0;
}

/* Best admissible neighbour; tabu[r] != 0 marks rank r tabu (nullable). */
int32_t oracle_eval_best(const int8_t *A, int32_t m, int32_t n, const int32_t *S, const int8_t *V,
                         int32_t k, const uint8_t *tabu, int64_t *best_f, int64_t *best_r, int32_t nthreads)
{
    if (k < 1 || k > ORACLE_KMAX || n < k) return -1;
    int64_t M = oracle_neighborhood_size(n, k);
    int32_t *until = NULL;
    if (tabu) {
        until = malloc(sizeof(int32_t) * (size_t)M);
        for (int64_t r = 0; r < M; r++) until[r] = tabu[r] ? 1 : 0; /* admissible at t=1 iff until < 1 */
    }
    packed_t P;
    pack_instance(A, m, n, S, &P);
    uint64_t *vb = malloc(sizeof(uint64_t) * (size_t)P.nw);
    pack_vector(V, n, vb);
    fr_t b = scan_neighbourhood(&P, vb, k, 1, NULL, until, 1, NULL, 0, nthreads, -1, NULL);
    *best_f = b.f == INT64_MAX ? -1 : b.f;
    *best_r = b.r;
    free(vb); free_packed(&P); free(until);
    return b.r < 0 ? -6 : 0;
}

/* ---------------------------------------------------------------------------------------
 * Tabu search, PAPER.md:241-258 (Section IV-B) after Taillard [11]; Fig. 1:
 * at each iteration the whole neighbourhood is generated and evaluated and the best candidate
 * replaces the current solution.
 *   - tabu list: FIFO of the last L accepted move ranks (reading R3), implemented literally as
 *     until[r]: a rank accepted at iteration t is tabu for t+1 .. t+L;
 *   - no aspiration by default (reading R4); with flags & 1 a tabu move is admissible when it is
 *     better than the best fitness seen so far (Taillard's criterion, variant R4');
 *   - with flags & 2 the tabu list holds visited SOLUTIONS instead of move ranks (variant R3',
 *     PAPER.md:243-244 read literally), see the solution set above;
 *     lowest rank wins ties (reading R5);
 *   - stop when f = 0 if stop_on_zero (checked before every iteration, also before t = 1),
 *     otherwise after `iters` iterations (reading R11).
 * res[0..5] = iters_done, final_f, best_f, best_iter, first_zero_iter (-1: never), solved.
 * ------------------------------------------------------------------------------------- */
int32_t oracle_tabu_run(const int8_t *A, int32_t m, int32_t n, const int32_t *S, int32_t k,
                        const int8_t *V0, int64_t iters, int64_t L, int32_t stop_on_zero,
                        int64_t *trace_r, int64_t *trace_f, int8_t *V_out, int64_t *res,
                        int32_t nthreads, int32_t flags)
{
    /* flags: 1 = aspiration (R4'), 2 = solution list (R3'): at iteration t the tabu list holds the
     * L most recently visited solutions V_{t-L} .. V_{t-1} (V_0 = the start, V_{t-1} = the current
     * solution, which is never a neighbour); a neighbour is tabu iff it equals one of them. */
    const int aspiration = flags & 1, solutions = (flags & 2) != 0;
    if (k < 1 || k > ORACLE_KMAX || n < k || m < 1 || iters < 0 || L < 0) return -1;
    int64_t M = oracle_neighborhood_size(n, k);
    if (L >= M) return -2;
    if (solutions && L < 1) return -1;
    packed_t P;
    pack_instance(A, m, n, S, &P);
    uint64_t *vb = malloc(sizeof(uint64_t) * (size_t)P.nw);
    int32_t *Y = malloc(sizeof(int32_t) * (size_t)m);
    int32_t *Hp = malloc(sizeof(int32_t) * (size_t)(n + 1));
    int32_t *until = calloc((size_t)M, sizeof(int32_t)); /* until[r] = 0: admissible from t = 1 */
    uint64_t *visited = NULL; /* V_s in slot s mod L */
    solset_t sols = { P.nw, 0, NULL };
    if (solutions) {
        visited = malloc(sizeof(uint64_t) * (size_t)P.nw * (size_t)L);
        sols.cap = 1;
        while (sols.cap < 2 * L) sols.cap <<= 1;
        sols.slot = malloc(sizeof(uint64_t *) * (size_t)sols.cap);
    }
    pack_vector(V0, n, vb);
    if (solutions) memcpy(visited, vb, sizeof(uint64_t) * (size_t)P.nw); /* V_0 */
    int64_t f = fitness_packed(&P, vb, Y, Hp);
    int64_t best_f = f, best_iter = 0, first_zero = (f == 0) ? 0 : -1, t;
    for (t = 1; t <= iters; t++) {
        if (stop_on_zero && f == 0) break;
        if (solutions) { /* the list of iteration t: V_s for max(0, t - L) <= s <= t - 1 */
            memset(sols.slot, 0, sizeof(uint64_t *) * (size_t)sols.cap);
            for (int64_t q = (t - L > 0 ? t - L : 0); q <= t - 1; q++)
                solset_insert(&sols, visited + (size_t)(q % L) * (size_t)P.nw);
        }
        fr_t b = scan_neighbourhood(&P, vb, k, 1, NULL, solutions ? NULL : until, t, NULL, 0, nthreads,
                                    aspiration ? best_f : -1, solutions ? &sols : NULL);
        if (b.r < 0) break; /* unreachable for L < M */
        /* apply: V <- V xor F_{r*}; flip set of r* found by walking the same nested loops */
        int32_t F[ORACLE_KMAX];
        oracle_flipsets(n, k, &b.r, 1, F);
        for (int32_t q = 0; q < k; q++) flip(vb, F[q]);
        f = b.f;
        until[b.r] = (int32_t)(t + L);
        if (solutions) memcpy(visited + (size_t)(t % L) * (size_t)P.nw, vb, sizeof(uint64_t) * (size_t)P.nw); /* V_t */
        if (trace_r) trace_r[t - 1] = b.r;
        if (trace_f) trace_f[t - 1] = b.f;
        if (f < best_f) { best_f = f; best_iter = t; }
        if (f == 0 && first_zero < 0) first_zero = t;
    }
    int64_t done = t - 1;
    if (V_out)
        for (int32_t i = 0; i < n; i++) V_out[i] = ((vb[i / 64] >> (i % 64)) & 1) ? -1 : 1;
    res[0] = done; res[1] = f; res[2] = best_f; res[3] = best_iter; res[4] = first_zero;
    res[5] = best_f == 0;
    free(vb); free(Y); free(Hp); free(until); free_packed(&P); free(visited); free(sols.slot);
    return 0;
}

int32_t oracle_max_threads(void)
{
#ifdef _OPENMP
    return omp_get_max_threads();
#else
    return 1;
#endif
}

/*
 * Plain-C use of the C ABI (include/lns.h), no Python or torch: build a planted PPP instance
 * (Definition 1) with its own splitmix64 stream, evaluate the 3-Hamming
 * neighbourhood once (lns_eval_neighborhood), run a tabu search (lns_tabu_run)
 * and a batch of restarts (lns_tabu_run_batch), all from host buffers; then the same search on the
 * second binary fitness, UBQP f(x) = x^T Q x (lns_bqp_*).
 *
 *   cc -O2 -I include examples/tabu_c.c -L paper_conf_ipps_luongmt10_b200 -llns \
 *      -Wl,-rpath,$PWD/paper_conf_ipps_luongmt10_b200 -o build/tabu_c && build/tabu_c [m n k iters]
 *
 * Exit code 0 when every call succeeds and the reported fitnesses are consistent.
 */
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>

#include "lns.h"

static uint64_t next(uint64_t *s)
{
    uint64_t z = (*s += 0x9E3779B97F4A7C15ULL);
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ULL;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBULL;
    return z ^ (z >> 31);
}

#define CHECK(call)                                                                      \
    do {                                                                                 \
        lns_status _s = (call);                                                          \
        if (_s != LNS_OK) {                                                              \
            fprintf(stderr, "%s: %s (%s)\n", #call, lns_strerror(_s), lns_last_error()); \
            return 1;                                                                    \
        }                                                                                \
    } while (0)

int main(int argc, char **argv)
{
    const int m = argc > 1 ? atoi(argv[1]) : 101, n = argc > 2 ? atoi(argv[2]) : 117;
    const int k = argc > 3 ? atoi(argv[3]) : 3;
    const int64_t iters = argc > 4 ? atoll(argv[4]) : 200;
    int8_t *A = malloc((size_t)m * n), *V = malloc(n), *Vout = malloc(n);
    int32_t *S = malloc(sizeof(int32_t) * m), *Y = malloc(sizeof(int32_t) * m);
    uint64_t s = 12345, w = 0;
    for (int64_t q = 0; q < (int64_t)m * n; q++) {  /* A: i.i.d. +-1 */
        if (q % 64 == 0) w = next(&s);
        A[q] = ((w >> (q % 64)) & 1) ? -1 : 1;
    }
    for (int i = 0; i < n; i++) {  /* the planted secret */
        if (i % 64 == 0) w = next(&s);
        V[i] = ((w >> (i % 64)) & 1) ? -1 : 1;
    }
    for (int j = 0; j < m; j++) {  /* rows negated so that A V* >= 0; S = A V* */
        int y = 0;
        for (int i = 0; i < n; i++) y += A[(int64_t)j * n + i] * V[i];
        if (y < 0) { for (int i = 0; i < n; i++) A[(int64_t)j * n + i] = -A[(int64_t)j * n + i]; y = -y; }
        S[j] = y;
    }
    lns_ctx *ctx = NULL;
    CHECK(lns_create(A, m, n, S, 0, &ctx));
    for (int i = 0; i < n; i += 3) V[i] = -V[i];  /* a start some flips away from the secret */
    for (int j = 0; j < m; j++) {
        int y = 0;
        for (int i = 0; i < n; i++) y += A[(int64_t)j * n + i] * V[i];
        Y[j] = y;
    }
    int64_t bf = -1, br = -1;
    CHECK(lns_eval_neighborhood(ctx, k, V, Y, NULL, &bf, &br, NULL));
    printf("C(%d,%d) = %lld neighbours: best f = %lld at rank %lld\n", n, k,
           (long long)lns_neighborhood_size(n, k), (long long)bf, (long long)br);
    lns_result r;
    int64_t *tr = malloc(sizeof(int64_t) * iters), *tf = malloc(sizeof(int64_t) * iters);
    CHECK(lns_tabu_run(ctx, k, iters, -1, 7, V, LNS_STOP_ON_ZERO, Vout, tr, tf, &r, NULL));
    printf("tabu search: %lld iterations, final f %lld, best f %lld (iteration %lld), solved %d, %.3f ms\n",
           (long long)r.iters_done, (long long)r.final_f, (long long)r.best_f, (long long)r.best_iter, r.solved,
           lns_last_kernel_ms(ctx));
    int ok = r.iters_done >= 1 && tf[0] == bf && tr[0] == br;  /* the first move is the evaluated best */
    lns_result rb[8];
    CHECK(lns_tabu_run_batch(ctx, k, 8, iters, -1, 99, NULL, 0, NULL, rb, NULL));
    for (int q = 0; q < 8; q++) ok &= rb[q].iters_done == iters && rb[q].best_f <= rb[q].final_f;
    printf("8 restarts x %lld iterations: best f of restart 0 = %lld, %.3f ms\n", (long long)iters,
           (long long)rb[0].best_f, lns_last_kernel_ms(ctx));
    lns_destroy(ctx);

    /* UBQP: symmetric Q with entries in [-100, 100] at density ~1/4, x0 = 0, 2-Hamming */
    const int32_t nq = n < 200 ? n : 200;
    int32_t *Q = calloc((size_t)nq * nq, sizeof(int32_t));
    uint8_t *x0 = calloc((size_t)nq, 1), *xo = malloc((size_t)nq);
    uint64_t sq = 2024;
    for (int32_t i = 0; i < nq; i++)
        for (int32_t j = i; j < nq; j++) {
            const uint64_t z = next(&sq);
            if ((z & 3) == 0) Q[(size_t)i * nq + j] = Q[(size_t)j * nq + i] = (int32_t)((z >> 8) % 201) - 100;
        }
    const int64_t Mq = lns_neighborhood_size(nq, 2);
    int32_t *fq = malloc(sizeof(int32_t) * (size_t)Mq);
    int64_t *trq = malloc(sizeof(int64_t) * 50), *tfq = malloc(sizeof(int64_t) * 50), rq[4];
    lns_bqp *bq = NULL;
    CHECK(lns_bqp_create(Q, nq, 0, &bq));
    CHECK(lns_bqp_eval_all(bq, 2, x0, fq, NULL));
    int64_t fmin = fq[0], rmin = 0;
    for (int64_t r2 = 1; r2 < Mq; r2++)
        if (fq[r2] < fmin) { fmin = fq[r2]; rmin = r2; }
    CHECK(lns_bqp_tabu_run(bq, 2, 50, -1, x0, xo, trq, tfq, rq, NULL));
    printf("UBQP n=%d, 2-Hamming: best neighbour of x0 f = %lld (rank %lld); 50 iterations: best f %lld, %.3f ms\n",
           nq, (long long)fmin, (long long)rmin, (long long)rq[2], lns_bqp_last_kernel_ms(bq));
    ok &= rq[0] == 50 && trq[0] == rmin && tfq[0] == fmin && rq[2] <= rq[1] && rq[2] <= fmin;
    lns_bqp_destroy(bq);
    free(Q); free(x0); free(xo); free(fq); free(trq); free(tfq);
    free(A); free(V); free(Vout); free(S); free(Y); free(tr); free(tf);
    printf(ok ? "ok\n" : "INCONSISTENT\n");
    return ok ? 0 : 2;
}

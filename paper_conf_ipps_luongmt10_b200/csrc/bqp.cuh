// bqp.cuh -- the k-Hamming tabu search on a second binary fitness: UBQP, f(x) = x^T Q x over
// x in {0,1}^n (SURVEY.md §8(f) f4 "a pluggable binary fitness"). Included at
// the end of lns.cu (same translation unit: shares fail / CK / DeviceGuard / pool_alloc).
//
// The paper's mappings are stated "for binary problems"; only the
// fitness changes. The neighbourhood, rank order (reading R6), tabu list (R3), selection (R5) and
// key packing are those of the PPP path. Incremental evaluation (derived in DESIGN.md §5.13):
// with g = Q x and d_i = 1 - 2 x_i, flipping F changes f by
//     sum_{i in F} h_i + 2 sum_{i<j in F} d_i d_j Q_ij,   h_i = 2 d_i g_i + Q_ii,
// so a neighbour costs k table reads and C(k,2) reads of Q (rows of the flip set, L1/L2
// resident); the move updates g with k rows of Q (g_j += sum_{i in F} d_i Q_ij).
namespace {

constexpr int BQ_NT = 256;      // eval CTA
constexpr int BQ_AT = 1024;     // init / apply CTA
constexpr int BQ_N_MAX = 4096;
// Keys span the whole u64 range (the biased fitness fills the high word), so "none" is all ones:
// a real key has r < 2^32 - 1 in its low word.
constexpr unsigned long long BQ_NONE = ~0ull;
enum { BS_F = 0, BS_T, BS_BEST, BS_BESTIT, BS_ERR, BS_N };  // state (int64); ERR: 1 bad x, 2 no move

__device__ __forceinline__ uint64_t bq_comb(uint64_t x, int e)
{
    return e == 1 ? x : e == 2 ? x * (x - 1) / 2 : x * (x - 1) * (x - 2) / 6;  // 0 for x < e
}

// Lexicographic unranking (reading R6) by the combinatorial number system:
// M - 1 - r = sum_e C(n-1-i_{K-e}, e); each term is the largest C(z, e) <= remainder (binary search).
template <int K>
__device__ __forceinline__ void bq_unrank(uint64_t r, int n, uint64_t M, int *idx)
{
    uint64_t R = M - 1 - r;
    int top = n - 1;
#pragma unroll
    for (int e = K; e >= 1; e--) {
        int lo = e - 1, hi = top;  // C(lo, e) = 0 <= R
        while (lo < hi) {
            const int mid = (lo + hi + 1) >> 1;
            if (bq_comb((uint64_t)mid, e) <= R) lo = mid; else hi = mid - 1;
        }
        idx[K - e] = n - 1 - lo;
        R -= bq_comb((uint64_t)lo, e);
        top = lo - 1;
    }
}

template <int K>
__device__ __forceinline__ void bq_succ(int n, int *idx)
{
    int i = K - 1;
    while (i > 0 && idx[i] == n - K + i) i--;
    idx[i]++;
#pragma unroll
    for (int j = 1; j < K; j++)
        if (j > i) idx[j] = idx[j - 1] + 1;
}

// Advance a sorted flip set by s ranks in lexicographic order (last index fastest): move the last
// index; each time it runs past n - 1 the prefix takes its own successor (a (K-1)-subset of
// [0, n - 2]) and the overshoot restarts after the new prefix. Exact for any s >= 0 that stays
// inside [0, M).
template <int K>
__device__ __forceinline__ bool bq_advance(int n, int *idx, int s)
{
    int c = idx[K - 1] + s;
    bool moved = false;
    if (K > 1) {
        while (c >= n) {
            const int over = c - n;
            int pre[K > 1 ? K - 1 : 1];
#pragma unroll
            for (int q = 0; q < K - 1; q++) pre[q] = idx[q];
            bq_succ<(K > 1 ? K - 1 : 1)>(n - 1, pre);
#pragma unroll
            for (int q = 0; q < K - 1; q++) idx[q] = pre[q];
            c = idx[K - 2] + 1 + over;
            moved = true;
        }
    }
    idx[K - 1] = c;
    return moved;
}

__device__ __forceinline__ unsigned long long bq_key(int32_t f, uint32_t r)
{
    return ((unsigned long long)((uint32_t)f ^ 0x80000000u) << 32) | r;  // order-preserving
}

// g = Q x, f = x^T g, state reset; x entries must be 0 or 1.
// Batched restarts (lns_bqp_tabu_run_batch): CTA r (init, apply) / grid row blockIdx.y = r (eval)
// works on restart r's slice of x, g, st, until and key; a single search is the grid of one row.
__global__ void __launch_bounds__(BQ_AT) k_bqp_init(const int32_t *__restrict__ Q, int n,
                                                    const uint8_t *__restrict__ x, int32_t *__restrict__ g,
                                                    int64_t *st)
{
    x += (size_t)blockIdx.x * n; g += (size_t)blockIdx.x * n; st += (size_t)blockIdx.x * BS_N;
    __shared__ unsigned long long s_f;
    __shared__ int s_bad;
    if (threadIdx.x == 0) { s_f = 0; s_bad = 0; }
    __syncthreads();
    long long part = 0;
    for (int j = threadIdx.x; j < n; j += blockDim.x) {
        int acc = 0;
        for (int i = 0; i < n; i++) acc += x[i] ? Q[(size_t)i * n + j] : 0;  // Q symmetric: column j
        g[j] = acc;
        if (x[j] > 1) s_bad = 1;
        part += x[j] ? (long long)acc : 0;
    }
    atomicAdd(&s_f, (unsigned long long)part);
    __syncthreads();
    if (threadIdx.x == 0) {
        const int64_t f = (int64_t)s_f;
        st[BS_F] = f; st[BS_T] = 0; st[BS_BEST] = f; st[BS_BESTIT] = 0; st[BS_ERR] = s_bad ? 1 : 0;
    }
}

// Tabu state of one search (reading R3: the FIFO of the last L accepted ranks), `S` words per
// restart: a bitmap of ceil(M/32) words (bit r set <=> rank r is tabu) followed by a ring of L
// ranks (slot (s - 1) mod L = the rank accepted at iteration s). The same list as an until[] array
// with until[r] = (iteration accepted) + L, at 1/32 of its memory traffic.

// Every neighbour of iteration t = st[T] + 1: fitness (fit_out, optional) and the least admissible
// key (tabu bit clear; tabu == nullptr: all admissible) MIN-reduced into *key.
template <int K>
__global__ void __launch_bounds__(BQ_NT) k_bqp_eval(const int32_t *__restrict__ Q, int n, uint64_t M,
                                                    const uint8_t *__restrict__ x, const int32_t *__restrict__ g,
                                                    const int64_t *__restrict__ st, const uint32_t *__restrict__ tabu,
                                                    uint64_t S, int32_t *__restrict__ fit_out, unsigned long long *key)
{
    extern __shared__ int32_t s_h[];  // h_i = 2 d_i g_i + Q_ii, then d_i (n + n ints)
    int32_t *s_d = s_h + n;
    __shared__ unsigned long long s_key;
    x += (size_t)blockIdx.y * n; g += (size_t)blockIdx.y * n; st += (size_t)blockIdx.y * BS_N; key += blockIdx.y;
    if (tabu) tabu += (size_t)blockIdx.y * S;
    if (st[BS_ERR]) return;  // uniform over the grid row
    for (int i = threadIdx.x; i < n; i += blockDim.x) {
        const int d = 1 - 2 * (int)x[i];
        s_d[i] = d;
        s_h[i] = 2 * d * g[i] + Q[(size_t)i * n + i];
    }
    if (threadIdx.x == 0) s_key = BQ_NONE;
    __syncthreads();
    const int32_t f0 = (int32_t)st[BS_F];
    // Warp-interleaved ranks: warp w owns [32 w per, 32 (w + 1) per) and lane l takes ranks
    // base + l + 32 j, so consecutive lanes hold consecutive ranks: the 32 ranks of a step are one
    // bitmap word (bit = lane), fit_out is coalesced, and (last index fastest) the Q row reads Q[a n + c], Q[b n + c] and the h[c], d[c]
    // table reads hit consecutive addresses across the warp.
    const uint64_t T = (uint64_t)gridDim.x * blockDim.x;
    const uint64_t per = (M + T - 1) / T;
    const uint64_t gw = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t lo = gw * 32 * per + (threadIdx.x & 31);
    const uint64_t hi = min(M, (gw + 1) * 32 * per);
    unsigned long long best = BQ_NONE;
    if (lo < hi) {
        int idx[K];
        bq_unrank<K>(lo, n, M, idx);
        // Flip set (a, b, c) in registers (c = the last index; (a, b) the prefix, k = 3; a alone,
        // k = 2). The prefix F \ {c} changes only when the run wraps: its part of the delta (pre),
        // its signs and its Q rows are kept in registers. Modular (u32) sums: every term fits int32
        // and so does f0 + delta (|f| <= sum |Q_ij| < 2^29), so the wrapped total is exact.
        int a = K >= 2 ? idx[0] : 0, b = K == 3 ? idx[1] : 0, c = idx[K - 1];
        uint32_t pre = 0;
        int dp0 = 0, dp1 = 0;
        const int32_t *q0 = Q, *q1 = Q;
        auto load_prefix = [&]() {
            if (K >= 2) { dp0 = s_d[a]; q0 = Q + (size_t)a * n; pre = (uint32_t)s_h[a]; }
            if (K == 3) {
                dp1 = s_d[b]; q1 = Q + (size_t)b * n;
                pre += (uint32_t)s_h[b] + (uint32_t)(2 * dp0 * dp1 * q0[b]);
            }
        };
        load_prefix();
        // least admissible (biased fitness, rank) of this lane: ranks only grow along the run, so a
        // strict "<" on the fitness keeps the lowest rank among equal fitnesses (reading R5)
        uint32_t bf = 0xffffffffu, br = 0xffffffffu;
        const uint32_t rhi = (uint32_t)hi;
        const uint32_t *wp = tabu ? tabu + (lo >> 5) : nullptr;  // bitmap word of r, advanced with r
        const unsigned lane = threadIdx.x & 31;
        for (uint32_t r = (uint32_t)lo;;) {
            uint32_t delta = pre + (uint32_t)s_h[c];
            if (K >= 2) {
                const int dc2 = 2 * s_d[c];
                delta += (uint32_t)(dc2 * dp0 * q0[c]);
                if (K == 3) delta += (uint32_t)(dc2 * dp1 * q1[c]);
            }
            const uint32_t fr = (uint32_t)f0 + delta;
            if (fit_out) fit_out[r] = (int32_t)fr;
            const uint32_t fb = fr ^ 0x80000000u;  // order-preserving for signed f
            if ((!wp || !((*wp >> lane) & 1u)) && fb < bf) { bf = fb; br = r; }
            if (rhi - r <= 32u) break;
            r += 32u;
            if (wp) ++wp;
            c += 32;
            if (K >= 2 && c >= n) {
                // the run passes the end of its prefix: the prefix takes its successor (a
                // (k-1)-subset of [0, n - 2]) and the overshoot restarts after it
                do {
                    const int over = c - n;
                    if (K == 2) {
                        ++a;
                        c = a + 1 + over;
                    } else {
                        if (b < n - 2) ++b; else { ++a; b = a + 1; }
                        c = b + 1 + over;
                    }
                } while (c >= n);
                load_prefix();
            }
        }
        if (br != 0xffffffffu) best = ((unsigned long long)bf << 32) | br;
    }
    best = warp_min_k(best);
    if ((threadIdx.x & 31) == 0 && best != BQ_NONE) atomicMin(&s_key, best);
    __syncthreads();
    if (threadIdx.x == 0 && s_key != BQ_NONE) atomicMin(key, s_key);
}

// Apply the winning move of iteration t = st[T] + 1: x ^= F, g += sum_{i in F} d_i Q_i., the tabu
// list (the rank accepted at t - L leaves, r enters), trace, best; *key reset for the next
// iteration. One CTA per search.
template <int K>
__global__ void __launch_bounds__(BQ_AT) k_bqp_apply(const int32_t *__restrict__ Q, int n, uint64_t M,
                                                     uint8_t *x, int32_t *g, int64_t *st, uint32_t *tabu,
                                                     uint64_t S, int64_t L, unsigned long long *key,
                                                     int64_t *trace_r, int64_t *trace_f)
{
    x += (size_t)blockIdx.x * n; g += (size_t)blockIdx.x * n; st += (size_t)blockIdx.x * BS_N; key += blockIdx.x;
    tabu += (size_t)blockIdx.x * S;
    if (st[BS_ERR]) return;
    const unsigned long long kv = *key;
    if (kv == BQ_NONE) {
        if (threadIdx.x == 0) st[BS_ERR] = 2;
        return;
    }
    const uint32_t r = (uint32_t)(kv & 0xffffffffu);
    const int32_t f = (int32_t)((uint32_t)(kv >> 32) ^ 0x80000000u);
    int idx[K], d[K];
    bq_unrank<K>(r, n, M, idx);
#pragma unroll
    for (int q = 0; q < K; q++) d[q] = 1 - 2 * (int)x[idx[q]];
    for (int j = threadIdx.x; j < n; j += blockDim.x) {
        int acc = g[j];
#pragma unroll
        for (int q = 0; q < K; q++) acc += d[q] * Q[(size_t)idx[q] * n + j];
        g[j] = acc;
    }
    __syncthreads();  // every thread has read x[F] before it flips
    if (threadIdx.x == 0) {
#pragma unroll
        for (int q = 0; q < K; q++) x[idx[q]] ^= 1;
        const int64_t t = st[BS_T] + 1;
        if (L > 0) {
            // tabu at iteration t' <=> accepted at t' - L .. t' - 1: for t + 1 the rank of t - L
            // leaves (it was tabu through t, so it is not r) and r enters; one writer per search
            uint32_t *ring = tabu + (M + 31) / 32;
            const size_t slot = (size_t)((t - 1) % L);
            if (t > L) {
                const uint32_t e = ring[slot];
                tabu[e >> 5] &= ~(1u << (e & 31));
            }
            tabu[r >> 5] |= 1u << (r & 31);
            ring[slot] = r;
        }
        if (trace_r) { trace_r[t - 1] = r; trace_f[t - 1] = f; }
        st[BS_F] = f; st[BS_T] = t;
        if (f < st[BS_BEST]) { st[BS_BEST] = f; st[BS_BESTIT] = t; }
        *key = BQ_NONE;
    }
}

}  // namespace

struct lns_bqp {
    int device = 0, n = 0, nsm = 148;
    int32_t *d_Q = nullptr, *d_g = nullptr, *d_fit = nullptr;
    uint8_t *d_x = nullptr;
    int64_t *d_st = nullptr, *d_tr = nullptr, *d_tf = nullptr;
    uint32_t *d_until = nullptr;  // tabu state(s): bitmap + ring per search (bq_tabu_words)
    unsigned long long *d_key = nullptr;
    size_t fit_cap = 0, until_cap = 0, tr_cap = 0;
    // batched restarts: R slices of x, g, state, key (the tabu states share d_until: R x S words)
    uint8_t *d_bx = nullptr;
    int32_t *d_bg = nullptr;
    int64_t *d_bst = nullptr;
    unsigned long long *d_bkey = nullptr;
    size_t bx_cap = 0, bg_cap = 0, bst_cap = 0, bkey_cap = 0;
    cudaStream_t st = nullptr;
    cudaEvent_t ev0 = nullptr, ev1 = nullptr, evu = nullptr;
    float last_ms = 0;
};

namespace {

lns_status bqp_check_k(const lns_bqp *c, int32_t k, uint64_t &M)
{
    if (!c) return fail(LNS_EINVAL, "null context");
    if (k < 1 || k > 3) return fail(LNS_EINVAL, "UBQP: k must be 1, 2 or 3");
    if (c->n < k) return fail(LNS_EINVAL, "n < k");
    M = (uint64_t)comb_k(c->n, k);
    if (M >= 0xffffffffull) return fail(LNS_ERANGE, "C(n,k) >= 2^32 - 1");
    return LNS_OK;
}

int bqp_blocks(const lns_bqp *c, uint64_t M)
{
    const uint64_t want = (M + BQ_NT - 1) / BQ_NT;
    return (int)std::max<uint64_t>(1, std::min<uint64_t>(want, (uint64_t)c->nsm * 8));
}

// 32-bit words of one search's tabu state: the bitmap and the ring of L ranks.
inline uint64_t bq_tabu_words(uint64_t M, int64_t L) { return (M + 31) / 32 + (uint64_t)L; }

// The buffers one launch works on: a single search (the context's own) or R batched restarts.
struct BqBufs {
    uint8_t *x;
    int32_t *g;
    int64_t *st;
    unsigned long long *key;
    uint32_t *until;
    int R;
};

BqBufs bq_single(lns_bqp *c) { return BqBufs{c->d_x, c->d_g, c->d_st, c->d_key, c->d_until, 1}; }

lns_status bqp_launch_eval(lns_bqp *c, int k, uint64_t M, uint64_t S, const BqBufs &b, const uint32_t *tabu, int32_t *fit)
{
    // one grid row per restart; R rows share the SMs (about 8 CTAs per SM in total)
    const int nb = b.R == 1 ? bqp_blocks(c, M)
                            : (int)std::max<uint64_t>(1, std::min<uint64_t>((M + BQ_NT - 1) / BQ_NT,
                                                                            ((uint64_t)c->nsm * 8 + b.R - 1) / b.R));
    const dim3 grid(nb, b.R);
    const size_t sm = 2 * sizeof(int32_t) * (size_t)c->n;
    switch (k) {
    case 1: k_bqp_eval<1><<<grid, BQ_NT, sm, c->st>>>(c->d_Q, c->n, M, b.x, b.g, b.st, tabu, S, fit, b.key); break;
    case 2: k_bqp_eval<2><<<grid, BQ_NT, sm, c->st>>>(c->d_Q, c->n, M, b.x, b.g, b.st, tabu, S, fit, b.key); break;
    default: k_bqp_eval<3><<<grid, BQ_NT, sm, c->st>>>(c->d_Q, c->n, M, b.x, b.g, b.st, tabu, S, fit, b.key); break;
    }
    CK(cudaGetLastError());
    return LNS_OK;
}

lns_status bqp_launch_apply(lns_bqp *c, int k, uint64_t M, uint64_t S, int64_t L, const BqBufs &b, bool trace)
{
    int64_t *tr = trace ? c->d_tr : nullptr, *tf = trace ? c->d_tf : nullptr;
    switch (k) {
    case 1: k_bqp_apply<1><<<b.R, BQ_AT, 0, c->st>>>(c->d_Q, c->n, M, b.x, b.g, b.st, b.until, S, L, b.key, tr, tf); break;
    case 2: k_bqp_apply<2><<<b.R, BQ_AT, 0, c->st>>>(c->d_Q, c->n, M, b.x, b.g, b.st, b.until, S, L, b.key, tr, tf); break;
    default: k_bqp_apply<3><<<b.R, BQ_AT, 0, c->st>>>(c->d_Q, c->n, M, b.x, b.g, b.st, b.until, S, L, b.key, tr, tf); break;
    }
    CK(cudaGetLastError());
    return LNS_OK;
}

// `iters` iterations of eval + apply on b: blocks of G = min(iters, 64) iterations captured once
// into a CUDA graph and replayed (every launch reads the iteration number from the device state),
// the remainder launched directly; ev0 is recorded after the graph is built (host work).
lns_status bqp_iterate(lns_bqp *c, int k, uint64_t M, int64_t L, int64_t iters, const BqBufs &b, bool trace)
{
    const uint64_t S = bq_tabu_words(M, L);
    lns_status s;
    const int64_t G = std::min<int64_t>(iters, 64);
    int64_t done = 0;
    bool timing_started = false;
    if (G > 0 && iters / G >= 2) {
        cudaGraph_t graph = nullptr;
        cudaGraphExec_t exec = nullptr;
        CK(cudaStreamBeginCapture(c->st, cudaStreamCaptureModeThreadLocal));
        for (int64_t q = 0; q < G; q++) {
            lns_status e1 = bqp_launch_eval(c, k, M, S, b, b.until, nullptr);
            lns_status e2 = e1 == LNS_OK ? bqp_launch_apply(c, k, M, S, L, b, trace) : e1;
            if (e2 != LNS_OK) { cudaStreamEndCapture(c->st, &graph); if (graph) cudaGraphDestroy(graph); return e2; }
        }
        CK(cudaStreamEndCapture(c->st, &graph));
        cudaError_t e = cudaGraphInstantiate(&exec, graph, 0);
        cudaGraphDestroy(graph);
        if (e != cudaSuccess) return fail(LNS_ECUDA, std::string("cudaGraphInstantiate: ") + cudaGetErrorString(e));
        CK(cudaEventRecord(c->ev0, c->st));
        timing_started = true;
        for (; done + G <= iters; done += G) {
            e = cudaGraphLaunch(exec, c->st);
            if (e != cudaSuccess) { cudaGraphExecDestroy(exec); return fail(LNS_ECUDA, cudaGetErrorString(e)); }
        }
        cudaGraphExecDestroy(exec);
    }
    if (!timing_started) CK(cudaEventRecord(c->ev0, c->st));
    for (; done < iters; done++) {
        if ((s = bqp_launch_eval(c, k, M, S, b, b.until, nullptr)) != LNS_OK) return s;
        if ((s = bqp_launch_apply(c, k, M, S, L, b, trace)) != LNS_OK) return s;
    }
    CK(cudaEventRecord(c->ev1, c->st));
    return LNS_OK;
}

// Order the private stream after the caller's stream (inputs the caller wrote there).
lns_status bqp_enter(lns_bqp *c, void *stream)
{
    CK(cudaEventRecord(c->evu, (cudaStream_t)stream));
    CK(cudaStreamWaitEvent(c->st, c->evu, 0));
    return LNS_OK;
}

lns_status bqp_start(lns_bqp *c, const uint8_t *x, const BqBufs &b)
{
    CK(cudaMemcpyAsync(b.x, x, (size_t)c->n * b.R, cudaMemcpyDefault, c->st));
    k_bqp_init<<<b.R, BQ_AT, 0, c->st>>>(c->d_Q, c->n, b.x, b.g, b.st);
    CK(cudaGetLastError());
    CK(cudaMemsetAsync(b.key, 0xff, sizeof(unsigned long long) * b.R, c->st));  // BQ_NONE = all ones
    return LNS_OK;
}

}  // namespace

extern "C" {

lns_status lns_bqp_create(const int32_t *Q, int32_t n, int32_t device, lns_bqp **out)
{
    if (!out || !Q) return fail(LNS_EINVAL, "null argument");
    *out = nullptr;
    if (n < 1) return fail(LNS_EINVAL, "n must be >= 1");
    if (n > BQ_N_MAX) return fail(LNS_ERANGE, "n > 4096");
    int ndev = 0;
    CK(cudaGetDeviceCount(&ndev));
    if (device < 0 || device >= ndev) return fail(LNS_EINVAL, "bad device index");
    std::vector<int32_t> hQ((size_t)n * n);  // Q may live on the host or on a device (UVA copy)
    CK(cudaMemcpy(hQ.data(), Q, sizeof(int32_t) * hQ.size(), cudaMemcpyDefault));
    Q = hQ.data();
    int64_t absum = 0;
    for (int64_t i = 0; i < n; i++)
        for (int64_t j = 0; j < n; j++) {
            const int32_t q = Q[i * n + j];
            if (q != Q[j * n + i]) return fail(LNS_EINVAL, "Q must be symmetric");
            absum += q < 0 ? -(int64_t)q : (int64_t)q;
        }
    // |f(x)|, |f(x')|, |g_i| and |Q_ii| are bounded by S = sum |Q_ij| < 2^29, so h_i (< 3 S),
    // the 2 Q_ij pair terms and every fitness fit int32 (the eval kernel sums them mod 2^32)
    if (absum >= ((int64_t)1 << 29)) return fail(LNS_ERANGE, "sum |Q_ij| >= 2^29");
    DeviceGuard dg(device);
    lns_bqp *c = new lns_bqp();
    c->device = device;
    c->n = n;
    cudaDeviceGetAttribute(&c->nsm, cudaDevAttrMultiProcessorCount, device);
    bool ok = pool_alloc(&c->d_Q, sizeof(int32_t) * (size_t)n * n) == cudaSuccess &&
              pool_alloc(&c->d_g, sizeof(int32_t) * (size_t)n) == cudaSuccess &&
              pool_alloc(&c->d_x, (size_t)n) == cudaSuccess &&
              pool_alloc(&c->d_st, sizeof(int64_t) * BS_N) == cudaSuccess &&
              pool_alloc(&c->d_key, sizeof(unsigned long long)) == cudaSuccess;
    if (!ok) { lns_bqp_destroy(c); return fail(LNS_ENOMEM, "cudaMalloc failed"); }
    if (cudaStreamCreateWithFlags(&c->st, cudaStreamNonBlocking) != cudaSuccess ||
        cudaEventCreate(&c->ev0) != cudaSuccess || cudaEventCreate(&c->ev1) != cudaSuccess ||
        cudaEventCreateWithFlags(&c->evu, cudaEventDisableTiming) != cudaSuccess) {
        lns_bqp_destroy(c);
        return fail(LNS_ECUDA, "stream / event creation failed");
    }
    if (cudaMemcpy(c->d_Q, Q, sizeof(int32_t) * (size_t)n * n, cudaMemcpyDefault) != cudaSuccess) {
        lns_bqp_destroy(c);
        return fail(LNS_ECUDA, "copy of Q failed");
    }
    *out = c;
    return LNS_OK;
}

void lns_bqp_destroy(lns_bqp *c)
{
    if (!c) return;
    DeviceGuard dg(c->device);
    if (c->st) cudaStreamSynchronize(c->st);
    pool_free(c->d_Q); pool_free(c->d_g); pool_free(c->d_x); pool_free(c->d_st); pool_free(c->d_key);
    pool_free(c->d_fit); pool_free(c->d_until); pool_free(c->d_tr); pool_free(c->d_tf);
    pool_free(c->d_bx); pool_free(c->d_bg); pool_free(c->d_bst); pool_free(c->d_bkey);
    if (c->ev0) cudaEventDestroy(c->ev0);
    if (c->ev1) cudaEventDestroy(c->ev1);
    if (c->evu) cudaEventDestroy(c->evu);
    if (c->st) cudaStreamDestroy(c->st);
    delete c;
}

lns_status lns_bqp_eval_all(lns_bqp *c, int32_t k, const uint8_t *x, int32_t *fitness_out, void *stream)
{
    uint64_t M;
    lns_status s = bqp_check_k(c, k, M);
    if (s != LNS_OK) return s;
    if (!x || !fitness_out) return fail(LNS_EINVAL, "null argument");
    DeviceGuard dg(c->device);
    if ((s = grow(c->d_fit, c->fit_cap, M)) != LNS_OK) return s;
    if ((s = bqp_enter(c, stream)) != LNS_OK) return s;
    if ((s = bqp_start(c, x, bq_single(c))) != LNS_OK) return s;
    CK(cudaEventRecord(c->ev0, c->st));
    if ((s = bqp_launch_eval(c, k, M, 0, bq_single(c), nullptr, c->d_fit)) != LNS_OK) return s;
    CK(cudaEventRecord(c->ev1, c->st));
    int64_t hs[BS_N];
    CK(cudaMemcpyAsync(hs, c->d_st, sizeof(hs), cudaMemcpyDeviceToHost, c->st));
    CK(cudaMemcpyAsync(fitness_out, c->d_fit, sizeof(int32_t) * M, cudaMemcpyDefault, c->st));
    CK(cudaStreamSynchronize(c->st));
    cudaEventElapsedTime(&c->last_ms, c->ev0, c->ev1);
    if (hs[BS_ERR] == 1) return fail(LNS_EINVAL, "x must be 0/1");
    return LNS_OK;
}

lns_status lns_bqp_tabu_run(lns_bqp *c, int32_t k, int64_t iters, int64_t tenure, const uint8_t *x0,
                            uint8_t *x_out, int64_t *trace_rank, int64_t *trace_fit, int64_t *res, void *stream)
{
    uint64_t M;
    lns_status s = bqp_check_k(c, k, M);
    if (s != LNS_OK) return s;
    if (!x0 || !res) return fail(LNS_EINVAL, "null argument");
    if (iters < 0 || iters >= ((int64_t)1 << 31)) return fail(LNS_EINVAL, "iters outside [0, 2^31)");
    const int64_t L = tenure < 0 ? (int64_t)(M / 6) : tenure;
    if ((uint64_t)L >= M) return fail(LNS_ERANGE, "tenure >= C(n,k)");
    if (iters + L >= ((int64_t)1 << 32) - 1) return fail(LNS_ERANGE, "iters + tenure >= 2^32");
    DeviceGuard dg(c->device);
    const bool trace = trace_rank || trace_fit;
    const uint64_t S = bq_tabu_words(M, L);
    if ((s = grow(c->d_until, c->until_cap, S)) != LNS_OK) return s;
    if (trace && c->tr_cap < (size_t)std::max<int64_t>(iters, 1)) {
        pool_free(c->d_tr); pool_free(c->d_tf);
        c->d_tr = c->d_tf = nullptr; c->tr_cap = 0;
        const size_t cap = (size_t)std::max<int64_t>(iters, 1);
        if (pool_alloc(&c->d_tr, 8 * cap) != cudaSuccess || pool_alloc(&c->d_tf, 8 * cap) != cudaSuccess)
            return fail(LNS_ENOMEM, "cudaMalloc failed");
        c->tr_cap = cap;
    }
    if ((s = bqp_enter(c, stream)) != LNS_OK) return s;
    CK(cudaMemsetAsync(c->d_until, 0, sizeof(uint32_t) * ((M + 31) / 32), c->st));  // the bitmap (the ring fills first)
    if ((s = bqp_start(c, x0, bq_single(c))) != LNS_OK) return s;
    if ((s = bqp_iterate(c, k, M, L, iters, bq_single(c), trace)) != LNS_OK) return s;
    int64_t hs[BS_N];
    CK(cudaMemcpyAsync(hs, c->d_st, sizeof(hs), cudaMemcpyDeviceToHost, c->st));
    if (x_out) CK(cudaMemcpyAsync(x_out, c->d_x, (size_t)c->n, cudaMemcpyDefault, c->st));
    CK(cudaStreamSynchronize(c->st));
    const int64_t nt = hs[BS_T];
    if (trace_rank && nt > 0) CK(cudaMemcpy(trace_rank, c->d_tr, 8 * (size_t)nt, cudaMemcpyDefault));
    if (trace_fit && nt > 0) CK(cudaMemcpy(trace_fit, c->d_tf, 8 * (size_t)nt, cudaMemcpyDefault));
    cudaEventElapsedTime(&c->last_ms, c->ev0, c->ev1);
    res[0] = nt; res[1] = hs[BS_F]; res[2] = hs[BS_BEST]; res[3] = hs[BS_BESTIT];
    if (hs[BS_ERR] == 1) return fail(LNS_EINVAL, "x0 must be 0/1");
    if (hs[BS_ERR] == 2) return fail(LNS_ENOADMISSIBLE, "every neighbour is tabu");
    return LNS_OK;
}

lns_status lns_bqp_tabu_run_batch(lns_bqp *c, int32_t k, int32_t R, int64_t iters, int64_t tenure,
                                  const uint8_t *x0s, uint8_t *x_outs, int64_t *res, void *stream)
{
    uint64_t M;
    lns_status s = bqp_check_k(c, k, M);
    if (s != LNS_OK) return s;
    if (!x0s || !res) return fail(LNS_EINVAL, "null argument");
    if (R < 1) return fail(LNS_EINVAL, "R must be >= 1");
    if (R > 65535) return fail(LNS_ERANGE, "R > 65535 (grid rows)");
    if (iters < 0 || iters >= ((int64_t)1 << 31)) return fail(LNS_EINVAL, "iters outside [0, 2^31)");
    const int64_t L = tenure < 0 ? (int64_t)(M / 6) : tenure;
    if ((uint64_t)L >= M) return fail(LNS_ERANGE, "tenure >= C(n,k)");
    if (iters + L >= ((int64_t)1 << 32) - 1) return fail(LNS_ERANGE, "iters + tenure >= 2^32");
    DeviceGuard dg(c->device);
    const size_t n = (size_t)c->n;
    const uint64_t S = bq_tabu_words(M, L);
    if ((s = grow(c->d_until, c->until_cap, S * (size_t)R)) != LNS_OK) return s;
    if ((s = grow(c->d_bx, c->bx_cap, n * R)) != LNS_OK) return s;
    if ((s = grow(c->d_bg, c->bg_cap, n * R)) != LNS_OK) return s;
    if ((s = grow(c->d_bst, c->bst_cap, (size_t)BS_N * R)) != LNS_OK) return s;
    if ((s = grow(c->d_bkey, c->bkey_cap, (size_t)R)) != LNS_OK) return s;
    const BqBufs b{c->d_bx, c->d_bg, c->d_bst, c->d_bkey, c->d_until, R};
    if ((s = bqp_enter(c, stream)) != LNS_OK) return s;
    CK(cudaMemset2DAsync(c->d_until, 4 * S, 0, 4 * ((M + 31) / 32), R, c->st));  // each restart's bitmap
    if ((s = bqp_start(c, x0s, b)) != LNS_OK) return s;
    if ((s = bqp_iterate(c, k, M, L, iters, b, false)) != LNS_OK) return s;
    std::vector<int64_t> hs((size_t)BS_N * R);
    CK(cudaMemcpyAsync(hs.data(), c->d_bst, sizeof(int64_t) * hs.size(), cudaMemcpyDeviceToHost, c->st));
    if (x_outs) CK(cudaMemcpyAsync(x_outs, c->d_bx, n * R, cudaMemcpyDefault, c->st));
    CK(cudaStreamSynchronize(c->st));
    cudaEventElapsedTime(&c->last_ms, c->ev0, c->ev1);
    int err = 0;
    for (int r = 0; r < R; r++) {
        const int64_t *h = hs.data() + (size_t)BS_N * r;
        res[4 * r] = h[BS_T]; res[4 * r + 1] = h[BS_F]; res[4 * r + 2] = h[BS_BEST]; res[4 * r + 3] = h[BS_BESTIT];
        if (h[BS_ERR] && !err) err = (int)h[BS_ERR];
    }
    if (err == 1) return fail(LNS_EINVAL, "x0s must be 0/1");
    if (err == 2) return fail(LNS_ENOADMISSIBLE, "every neighbour is tabu");
    return LNS_OK;
}

double lns_bqp_last_kernel_ms(const lns_bqp *c) { return c ? (double)c->last_ms : -1.0; }

}  // extern "C"

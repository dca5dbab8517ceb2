// lns.cu -- sm_100a kernels and C ABI (include/lns.h) of the k-Hamming tabu search on the
// Permuted Perceptron Problem (Luong, Melab, Talbi, LSPP@IPDPS 2010; PAPER.md).
//
// Design:
//  * A is bit-packed once (sign bits, bit = 1 <=> -1). Per iteration every CTA builds, in shared
//    memory, a "plan" of the current state: rows sorted by Y (counting sort over the lattice
//    Y = vmin + 2u), the sign bits X = (A o V)'s "-1" indicator permuted into that row order and
//    stored [row-word][column], the segment boundaries of equal-Y rows, and per-bin constants.
//  * A neighbour F = {a<b<c} moves row j to Y'_j = Y_j - 2k + 4 t_j, t_j = #{i in F : x_ji = 1}
//    (PAPER.md:227-229 with V' = V xor F). All rows of one Y-segment land in the same k+1 bins, so
//    the new histogram H' only needs, per segment, how many rows have t = 0..k.
//    Those counts come from bit-sliced t (LOP3) and POPC over the segment's row words; a sliding
//    window over the segment lattice turns them into H'(b) and the fitness (30-weighted penalty on
//    negative bins, |H - H'| on bins 0..n), exactly, in integers.
//  * Ranks are lexicographic (reading R6); each lane unranks exactly (integer combinatorial number
//    system, float estimate + integer correction). The (fitness, rank) pair is packed into one
//    63-bit key, so a u64 MIN gives "least fitness, lowest rank" (reading R5) at warp, CTA, grid and
//    (NCCL) multi-GPU level.
//  * The whole tabu search runs in ONE persistent cooperative kernel: one grid barrier per
//    iteration; every CTA applies the winning move to its own shared-memory copy of (V, Y).
#include "lns.h"

#include <cuda_runtime.h>
#include <dlfcn.h>

#include <climits>
#include <cmath>
#include <cstdio>
#include <cstring>
#include <string>
#include <vector>

#define LNS_VERSION_NUM 100

namespace {

constexpr int64_t KEY_NONE = INT64_MAX;
constexpr int NT = 512;           // threads per CTA
constexpr int NWARP = NT / 32;
constexpr unsigned FULL = 0xffffffffu;

thread_local std::string g_err;

// ------------------------------------------------------------------------------------------
// Device data
// ------------------------------------------------------------------------------------------
struct DevInst {
    int32_t m, n, W, NWn;      // W = ceil(m/32) row words, NWn = ceil(n/32) column words
    const uint32_t *Arow;      // m x NWn, bit (i%32) of word i/32 = 1 <=> A[j][i] = -1
    const int32_t *H;          // n+1 bins of S
};

// fstate layout (int64): current f, iterations done, best f, best iter, first zero iter, done, error
enum { FS_F = 0, FS_T, FS_BEST, FS_BESTIT, FS_ZERO, FS_DONE, FS_ERR, FS_N };

struct SearchArgs {
    DevInst I;
    uint32_t M;          // C(n,k)
    uint32_t lo, hi;     // rank slice of this device
    int64_t iters;       // iterations to run (persistent) / capacity (stepped)
    int64_t L;           // tenure
    int32_t stop_on_zero;
    uint32_t *vb;        // state: NWn words of V's sign bits
    int32_t *Y;          // state: m
    int64_t *fs;         // FS_N
    uint32_t *tabu;      // ceil(M/32) words (only this device's slice is used)
    uint32_t *ring;      // L+1 entries: rank accepted at iteration t sits in ring[t % (L+1)]
    int64_t *keys;       // 3 slots (persistent) / accumulator (stepped)
    unsigned *bar;       // grid barrier (count, generation) / stepped: last-block counter
    int64_t *trace_r, *trace_f;
};

// Shared-memory carve-up (identical on host and device).
struct Smem {
    int X, Y, vb, H, seg, cur, rowAt, bins, total;
};

__host__ __device__ inline int align16(int x) { return (x + 15) & ~15; }

__host__ __device__ inline Smem smem_layout(int m, int n, int W, int NWn, int K)
{
    Smem s;
    int o = 0;
    s.X = o;     o = align16(o + 4 * W * n);
    s.Y = o;     o = align16(o + 4 * m);
    s.vb = o;    o = align16(o + 4 * NWn);
    s.H = o;     o = align16(o + 4 * (n + 1));
    s.seg = o;   o = align16(o + 4 * (n + 4));          // Upad + 1 <= n + 3
    s.cur = o;   o = align16(o + 4 * (n + 4));
    s.rowAt = o; o = align16(o + 4 * m);
    s.bins = o;  o = align16(o + 8 * (n + 4 + 2 * K));  // Upad + 2K bins
    s.total = o;
    return s;
}

struct PlanScalars {
    int vmin, Upad, base;
    int64_t key;
    int red[2 * NWARP + 2];
    unsigned long long redk[NWARP];
};

__device__ __forceinline__ uint64_t C2(uint64_t y) { return y * (y - 1) / 2; }
__device__ __forceinline__ uint64_t C3(uint64_t z) { return z * (z - 1) * (z - 2) / 6; }

// Exact lexicographic unranking (reading R6) via the complement identity
// lex_rank(a<b<c) = M - 1 - [C(n-1-a,3) + C(n-1-b,2) + C(n-1-c,1)] (combinatorial number system).
// Float estimates are corrected by exact 64-bit integer comparisons, so the result is exact for
// every n allowed by the limits (C(n,3) < 2^32).
template <int K>
__device__ __forceinline__ void unrank(uint32_t r, int n, uint32_t M, int &a, int &b, int &c)
{
    if (K == 1) { a = (int)r; b = -1; c = -1; return; }
    uint64_t R = (uint64_t)(M - 1u - r);
    int top = n - 1;
    if (K == 3) {
        int z = (int)cbrtf(6.0f * (float)R) + 1;
        z = min(max(z, 2), top);
        while (C3(z) > R) z--;
        while (z + 1 <= top && C3(z + 1) <= R) z++;
        R -= C3(z);
        a = n - 1 - z;
        top = z - 1;
    }
    int y = (int)((1.0f + sqrtf(8.0f * (float)R + 1.0f)) * 0.5f);
    y = min(max(y, 1), top);
    while (C2(y) > R) y--;
    while (y + 1 <= top && C2(y + 1) <= R) y++;
    R -= C2(y);
    if (K == 2) { a = n - 1 - y; b = n - 1 - (int)R; c = -1; }
    else { b = n - 1 - y; c = n - 1 - (int)R; }
}

__device__ __forceinline__ int warp_min_i(int v) {
    for (int o = 16; o; o >>= 1) v = min(v, __shfl_xor_sync(FULL, v, o));
    return v;
}
__device__ __forceinline__ int warp_max_i(int v) {
    for (int o = 16; o; o >>= 1) v = max(v, __shfl_xor_sync(FULL, v, o));
    return v;
}
__device__ __forceinline__ int warp_sum_i(int v) {
    for (int o = 16; o; o >>= 1) v += __shfl_xor_sync(FULL, v, o);
    return v;
}
__device__ __forceinline__ unsigned long long warp_min_k(unsigned long long v) {
    for (int o = 16; o; o >>= 1) {
        unsigned long long w = __shfl_xor_sync(FULL, v, o);
        v = w < v ? w : v;
    }
    return v;
}

// Block-wide min of a key; result valid in all threads.
__device__ unsigned long long block_min_key(unsigned long long v, PlanScalars &ps)
{
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    v = warp_min_k(v);
    if (lane == 0) ps.redk[warp] = v;
    __syncthreads();
    if (warp == 0) {
        unsigned long long w = lane < NWARP ? ps.redk[lane] : (unsigned long long)KEY_NONE;
        w = warp_min_k(w);
        if (lane == 0) ps.key = (int64_t)w;
    }
    __syncthreads();
    return (unsigned long long)ps.key;
}

// ------------------------------------------------------------------------------------------
// Plan: per-iteration shared-memory structures of the current state (Y, V).
// ------------------------------------------------------------------------------------------
template <int K>
__device__ void build_plan(const DevInst &I, unsigned char *sm, const Smem &L, PlanScalars &ps)
{
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int m = I.m, n = I.n;
    const int *Ys = (const int *)(sm + L.Y);
    const uint32_t *vbs = (const uint32_t *)(sm + L.vb);
    const int *Hs = (const int *)(sm + L.H);
    int *seg = (int *)(sm + L.seg);
    int *cur = (int *)(sm + L.cur);
    int *rowAt = (int *)(sm + L.rowAt);
    int2 *bins = (int2 *)(sm + L.bins);
    uint32_t *X = (uint32_t *)(sm + L.X);

    // 1. value range of Y. (Written with min and max, not min(-y): nvcc 12.9 miscompiled the
    //    unrolled "mx = min(mx, -y)" into a 3-input min that dropped one negation.)
    int mn = INT_MAX, mx = INT_MIN;
    for (int j = tid; j < m; j += NT) { int y = Ys[j]; mn = min(mn, y); mx = max(mx, y); }
    mn = warp_min_i(mn); mx = warp_max_i(mx);
    if (lane == 0) { ps.red[warp] = mn; ps.red[NWARP + warp] = mx; }
    __syncthreads();
    if (warp == 0) {
        int a = lane < NWARP ? ps.red[lane] : INT_MAX, b = lane < NWARP ? ps.red[NWARP + lane] : INT_MIN;
        a = warp_min_i(a); b = warp_max_i(b);
        if (lane == 0) {
            int U = (b - a) / 2 + 1;
            ps.vmin = a;
            ps.Upad = (U + 1) & ~1;
        }
    }
    __syncthreads();
    const int vmin = ps.vmin, Upad = ps.Upad, NB = Upad + 2 * K;
    // 2. counting sort over the lattice u = (y - vmin)/2
    for (int u = tid; u <= Upad; u += NT) seg[u] = 0;
    __syncthreads();
    for (int j = tid; j < m; j += NT) atomicAdd(&seg[(Ys[j] - vmin) >> 1], 1);
    // bins: bin beta <-> value b = vmin + 2(beta - K); cost(h) = |h - Hb| + wb h
    int hsum = 0;
    for (int beta = tid; beta < NB; beta += NT) {
        int b = vmin + 2 * (beta - K);
        int2 bn;
        if (b < 0) bn = make_int2(0, 60 * (-b) - 1);     // 30 (|y| - y) = 60 |y| for y < 0
        else if (b <= n) { bn = make_int2(Hs[b], 0); hsum += Hs[b]; }
        else bn = make_int2(0, 0);
        bins[beta] = bn;
    }
    hsum = warp_sum_i(hsum);
    if (lane == 0) ps.red[warp] = hsum;
    __syncthreads();
    // 3. exclusive scan of the counts (warp 0), base = m - (H mass inside the bin window)
    if (warp == 0) {
        int run = 0;
        for (int b0 = 0; b0 <= Upad; b0 += 32) {
            int u = b0 + lane;
            int v = (u < Upad) ? seg[u] : 0;
            int inc = v;
            for (int o = 1; o < 32; o <<= 1) { int t = __shfl_up_sync(FULL, inc, o); if (lane >= o) inc += t; }
            if (u <= Upad) { seg[u] = run + inc - v; cur[u] = run + inc - v; }
            run += __shfl_sync(FULL, inc, 31);
        }
        int hs = lane < NWARP ? ps.red[lane] : 0;
        hs = warp_sum_i(hs);
        if (lane == 0) ps.base = m - hs;
    }
    __syncthreads();
    // 4. place rows
    for (int j = tid; j < m; j += NT) {
        int p = atomicAdd(&cur[(Ys[j] - vmin) >> 1], 1);
        rowAt[p] = j;
    }
    __syncthreads();
    // 5. X[w][c] = bits x_{rowAt[32w+l], c} (x = 1 <=> A_jc V_c = -1), one warp per row word
    for (int w = warp; w < I.W; w += NWARP) {
        int p = 32 * w + lane;
        bool valid = p < m;
        const uint32_t *ar = I.Arow + (size_t)(valid ? rowAt[p] : 0) * I.NWn;
        for (int cw = 0; cw < I.NWn; cw++) {
            uint32_t word = valid ? (__ldg(ar + cw) ^ vbs[cw]) : 0u;
            uint32_t mine = 0;
#pragma unroll
            for (int cc = 0; cc < 32; cc++) {
                uint32_t bal = __ballot_sync(FULL, (word >> cc) & 1u);
                if (lane == cc) mine = bal;
            }
            int c = 32 * cw + lane;
            if (c < n) X[w * n + c] = mine;
        }
    }
    __syncthreads();
}

// Fitness of neighbour (a, b, c) from the plan (exact; see file header).
template <int K>
__device__ __forceinline__ int eval_fit(const uint32_t *__restrict__ X, const int *__restrict__ seg,
                                        const int2 *__restrict__ bins, int n, int Upad, int base,
                                        int a, int b, int c)
{
    int f = base;
    int ce[K], co[K];
#pragma unroll
    for (int q = 0; q < K; q++) { ce[q] = 0; co[q] = 0; }
    int st = seg[0];
    for (int u = 0; u < Upad + 2 * K; u += 2) {
#pragma unroll
        for (int par = 0; par < 2; par++) {
            const int uu = u + par;
            int en = (uu < Upad) ? seg[uu + 1] : st;
            int c1 = 0, c2 = 0, c3 = 0;
            if (st < en) {
                const int w0 = st >> 5, w1 = (en - 1) >> 5;
                for (int w = w0; w <= w1; w++) {
                    uint32_t mask = FULL;
                    if (w == w0) mask &= FULL << (st & 31);
                    if (w == w1) mask &= FULL >> (31 - ((en - 1) & 31));
                    const uint32_t *xr = X + w * n;
                    uint32_t xa = xr[a];
                    if (K == 1) {
                        c1 += __popc(xa & mask);
                    } else if (K == 2) {
                        uint32_t xb = xr[b];
                        c1 += __popc((xa ^ xb) & mask);
                        c2 += __popc((xa & xb) & mask);
                    } else {
                        uint32_t xb = xr[b], xc = xr[c];
                        uint32_t lo = xa ^ xb ^ xc;
                        uint32_t hi = (xa & xb) | (xc & (xa ^ xb));
                        c1 += __popc(lo & mask);
                        c2 += __popc(hi & mask);
                        c3 += __popc(lo & hi & mask);
                    }
                }
            }
            // N_t = rows of this segment with t flipped "-1" entries; they land in bin uu + 2t
            int N[K + 1];
            const int len = en - st;
            if (K == 1) { N[1] = c1; N[0] = len - c1; }
            else if (K == 2) { N[2] = c2; N[1] = c1; N[0] = len - c1 - c2; }
            else { N[3] = c3; N[2] = c2 - c3; N[1] = c1 - c3; N[0] = len - c1 - c2 + c3; }
            int h;
            int *ch = par ? co : ce;
            h = ch[0] + N[0];
#pragma unroll
            for (int q = 0; q < K - 1; q++) ch[q] = ch[q + 1] + N[q + 1];
            ch[K - 1] = N[K];
            const int2 bn = bins[uu];
            f += abs(h - bn.x) + bn.y * h;
            st = en;
        }
    }
    return f;
}

__device__ __forceinline__ uint32_t ldcg_u32(const uint32_t *p) { return __ldcg(p); }

// Evaluate ranks [blo, bhi) (blo 32-aligned) of this CTA; returns this thread's best key.
template <int K, bool WRITE_ALL>
__device__ unsigned long long eval_range(const DevInst &I, const unsigned char *sm, const Smem &L,
                                         const PlanScalars &ps, uint32_t M, uint32_t blo, uint32_t bhi,
                                         const uint32_t *tabu, int32_t *fit_out)
{
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const uint32_t *X = (const uint32_t *)(sm + L.X);
    const int *seg = (const int *)(sm + L.seg);
    const int2 *bins = (const int2 *)(sm + L.bins);
    const int Upad = ps.Upad, base = ps.base;
    unsigned long long best = (unsigned long long)KEY_NONE;
    for (uint32_t r0 = blo + 32u * warp; r0 < bhi; r0 += NT) {
        const uint32_t r = r0 + lane;
        if (r < bhi) {
            bool is_tabu = false;
            if (tabu) is_tabu = (ldcg_u32(tabu + (r >> 5)) >> (r & 31)) & 1u;
            if (!is_tabu || WRITE_ALL) {
                int a, b, c;
                unrank<K>(r, I.n, M, a, b, c);
                int f = eval_fit<K>(X, seg, bins, I.n, Upad, base, a, b, c);
                if (WRITE_ALL) fit_out[r] = f;
                unsigned long long key = ((unsigned long long)(uint32_t)f << 32) | r;
                if (!is_tabu && key < best) best = key;
            }
        }
    }
    return best;
}

// Apply the move F to the CTA's shared copy of (Y, V): Y'_j = Y_j - 2 sum_{i in F} B_ji,
// B_ji = V_i A_ji, then flip the bits of V.
template <int K>
__device__ void apply_move(const DevInst &I, int *Ys, uint32_t *vbs, int a, int b, int c)
{
    for (int j = threadIdx.x; j < I.m; j += NT) {
        const uint32_t *ar = I.Arow + (size_t)j * I.NWn;
        int d = (((__ldg(ar + (a >> 5)) ^ vbs[a >> 5]) >> (a & 31)) & 1u) ? -1 : 1;
        if (K >= 2) d += (((__ldg(ar + (b >> 5)) ^ vbs[b >> 5]) >> (b & 31)) & 1u) ? -1 : 1;
        if (K == 3) d += (((__ldg(ar + (c >> 5)) ^ vbs[c >> 5]) >> (c & 31)) & 1u) ? -1 : 1;
        Ys[j] -= 2 * d;
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        vbs[a >> 5] ^= 1u << (a & 31);
        if (K >= 2) vbs[b >> 5] ^= 1u << (b & 31);
        if (K == 3) vbs[c >> 5] ^= 1u << (c & 31);
    }
    __syncthreads();
}

__device__ __forceinline__ void grid_barrier(unsigned *bar, unsigned nblocks)
{
    __syncthreads();
    if (threadIdx.x == 0) {
        volatile unsigned *gen = bar + 1;
        unsigned g = *gen;
        __threadfence();
        unsigned arrived = atomicAdd(bar, 1u);
        if (arrived == nblocks - 1) {
            atomicExch(bar, 0u);
            __threadfence();
            atomicAdd(bar + 1, 1u);
        } else {
            while (*gen == g) { }
        }
        __threadfence();
    }
    __syncthreads();
}

// Slice [blo, bhi) of CTA `b` of `nb` inside [lo, hi), boundaries on multiples of 32.
__device__ __forceinline__ void cta_slice(uint32_t lo, uint32_t hi, unsigned b, unsigned nb, uint32_t &blo, uint32_t &bhi)
{
    uint64_t span = hi - lo;
    blo = lo + 32u * (uint32_t)((span * b / nb) / 32);
    bhi = (b + 1 == nb) ? hi : lo + 32u * (uint32_t)((span * (b + 1) / nb) / 32);
}

__device__ void load_state(const SearchArgs &A, unsigned char *sm, const Smem &L)
{
    int *Ys = (int *)(sm + L.Y);
    uint32_t *vbs = (uint32_t *)(sm + L.vb);
    int *Hs = (int *)(sm + L.H);
    for (int j = threadIdx.x; j < A.I.m; j += NT) Ys[j] = A.Y[j];
    for (int w = threadIdx.x; w < A.I.NWn; w += NT) vbs[w] = A.vb[w];
    for (int b = threadIdx.x; b <= A.I.n; b += NT) Hs[b] = A.I.H[b];
    __syncthreads();
}

// ------------------------------------------------------------------------------------------
// Kernels
// ------------------------------------------------------------------------------------------

// Initial state: V0 (int8 +-1) -> sign bits, Y = A V0, f from scratch. One CTA.
// If Ycheck != nullptr the given Y must equal A V0 (else FS_ERR = 1).
__global__ void __launch_bounds__(NT) k_init(DevInst I, const int8_t *V0, uint32_t *vb, int32_t *Y,
                                             const int32_t *Ycheck, int64_t *fs)
{
    __shared__ int hist[4096 + 1];
    __shared__ int s_bad;
    __shared__ long long s_pen;
    const int tid = threadIdx.x;
    if (tid == 0) { s_bad = 0; s_pen = 0; }
    for (int w = tid; w < I.NWn; w += NT) {
        uint32_t word = 0;
        for (int q = 0; q < 32; q++) {
            int i = 32 * w + q;
            if (i < I.n) {
                int8_t v = V0[i];
                if (v != 1 && v != -1) s_bad = 1;
                if (v < 0) word |= 1u << q;
            }
        }
        vb[w] = word;
    }
    const bool use_hist = I.n <= 4096;
    for (int b = tid; b <= I.n && use_hist; b += NT) hist[b] = 0;
    __syncthreads();
    long long pen = 0;
    for (int j = tid; j < I.m; j += NT) {
        const uint32_t *ar = I.Arow + (size_t)j * I.NWn;
        int d = 0;
        for (int w = 0; w < I.NWn; w++) d += __popc(__ldg(ar + w) ^ vb[w]);
        int y = I.n - 2 * d;  // <a_j, v> = n - 2 popcount(a xor v)
        Y[j] = y;
        if (Ycheck && Ycheck[j] != y) s_bad = 1;
        if (y < 0) pen += -2 * (long long)y;
        if (y >= 0 && y <= I.n && use_hist) atomicAdd(&hist[y], 1);
    }
    atomicAdd((unsigned long long *)&s_pen, (unsigned long long)pen);
    __syncthreads();
    int hd = 0;
    for (int b = tid; b <= I.n && use_hist; b += NT) hd += abs(I.H[b] - hist[b]);
    __shared__ int s_hd;
    if (tid == 0) s_hd = 0;
    __syncthreads();
    atomicAdd(&s_hd, hd);
    __syncthreads();
    if (tid == 0) {
        int64_t f = 30 * (int64_t)s_pen + s_hd;
        fs[FS_F] = f; fs[FS_T] = 0; fs[FS_BEST] = f; fs[FS_BESTIT] = 0;
        fs[FS_ZERO] = (f == 0) ? 0 : -1; fs[FS_DONE] = 0; fs[FS_ERR] = (s_bad || !use_hist) ? 1 : 0;
    }
}

// The persistent tabu search: all iterations in one cooperative launch.
template <int K>
__global__ void __launch_bounds__(NT, 1) k_search(SearchArgs A)
{
    extern __shared__ __align__(16) unsigned char sm[];
    __shared__ PlanScalars ps;
    const Smem L = smem_layout(A.I.m, A.I.n, A.I.W, A.I.NWn, K);
    int *Ys = (int *)(sm + L.Y);
    uint32_t *vbs = (uint32_t *)(sm + L.vb);
    const unsigned nb = gridDim.x, bid = blockIdx.x;
    const bool leader = (bid == 0 && threadIdx.x == 0);
    load_state(A, sm, L);
    uint32_t blo, bhi;
    cta_slice(A.lo, A.hi, bid, nb, blo, bhi);
    int64_t f = A.fs[FS_F];
    int64_t best_f = A.fs[FS_BEST], best_it = A.fs[FS_BESTIT], zero_it = A.fs[FS_ZERO];
    const int64_t t0 = A.fs[FS_T];
    int64_t t = t0 + 1;
    bool failed = false;
    for (; t <= t0 + A.iters; t++) {
        if (A.stop_on_zero && f == 0) break;
        build_plan<K>(A.I, sm, L, ps);
        unsigned long long mine = eval_range<K, false>(A.I, sm, L, ps, A.M, blo, bhi, A.L > 0 ? A.tabu : nullptr, nullptr);
        unsigned long long bk = block_min_key(mine, ps);
        if (threadIdx.x == 0 && bk != (unsigned long long)KEY_NONE)
            atomicMin((unsigned long long *)&A.keys[t % 3], bk);
        grid_barrier(A.bar, nb);
        if (threadIdx.x == 0) ps.key = (int64_t)__ldcg((const unsigned long long *)&A.keys[t % 3]);
        if (leader) A.keys[(t + 2) % 3] = KEY_NONE;
        __syncthreads();
        const int64_t key = ps.key;
        if (key == KEY_NONE) { failed = true; break; }
        const uint32_t r = (uint32_t)(key & 0xffffffffu);
        f = key >> 32;
        int a, b, c;
        unrank<K>(r, A.I.n, A.M, a, b, c);
        apply_move<K>(A.I, Ys, vbs, a, b, c);
        if (threadIdx.x == 0 && A.L > 0) {
            const int64_t R1 = A.L + 1;
            if (t > A.L) {
                uint32_t old = __ldcg(&A.ring[(t - A.L) % R1]);
                if (old >= blo && old < bhi) atomicAnd(&A.tabu[old >> 5], ~(1u << (old & 31)));
            }
            if (r >= blo && r < bhi) atomicOr(&A.tabu[r >> 5], 1u << (r & 31));
            if (bid == 0) { A.ring[t % R1] = r; __threadfence(); }
        }
        if (leader) {
            if (A.trace_r) A.trace_r[t - 1] = r;
            if (A.trace_f) A.trace_f[t - 1] = f;
            if (f < best_f) { best_f = f; best_it = t; }
            if (f == 0 && zero_it < 0) zero_it = t;
        }
    }
    if (bid == 0) {
        for (int j = threadIdx.x; j < A.I.m; j += NT) A.Y[j] = Ys[j];
        for (int w = threadIdx.x; w < A.I.NWn; w += NT) A.vb[w] = vbs[w];
        if (threadIdx.x == 0) {
            A.fs[FS_F] = f; A.fs[FS_T] = t - 1; A.fs[FS_BEST] = best_f; A.fs[FS_BESTIT] = best_it;
            A.fs[FS_ZERO] = zero_it; A.fs[FS_DONE] = (A.stop_on_zero && f == 0) ? 1 : 0;
            if (failed) A.fs[FS_ERR] = 2;
        }
    }
}

// Stepped mode, evaluation: partial best key of this device's slice into key_out[0].
// The last CTA to finish publishes the accumulator and resets it (no extra launch).
template <int K, bool WRITE_ALL>
__global__ void __launch_bounds__(NT, 1) k_step_eval(SearchArgs A, int64_t *key_out, int32_t *fit_out)
{
    extern __shared__ __align__(16) unsigned char sm[];
    __shared__ PlanScalars ps;
    __shared__ bool s_last;
    const Smem L = smem_layout(A.I.m, A.I.n, A.I.W, A.I.NWn, K);
    if (!WRITE_ALL && A.fs[FS_DONE]) {
        if (blockIdx.x == 0 && threadIdx.x == 0) *key_out = KEY_NONE;
        return;
    }
    load_state(A, sm, L);
    uint32_t blo, bhi;
    cta_slice(A.lo, A.hi, blockIdx.x, gridDim.x, blo, bhi);
    build_plan<K>(A.I, sm, L, ps);
    unsigned long long mine = eval_range<K, WRITE_ALL>(A.I, sm, L, ps, A.M, blo, bhi, A.tabu, fit_out);
    unsigned long long bk = block_min_key(mine, ps);
    if (threadIdx.x == 0) {
        if (bk != (unsigned long long)KEY_NONE) atomicMin((unsigned long long *)A.keys, bk);
        __threadfence();
        unsigned done = atomicAdd(A.bar, 1u);
        s_last = (done == gridDim.x - 1);
        if (s_last) {
            __threadfence();
            *key_out = (int64_t)atomicExch((unsigned long long *)A.keys, (unsigned long long)KEY_NONE);
            A.bar[0] = 0;
        }
    }
}

// Stepped mode, move: key[0] is the global minimum. One CTA.
template <int K>
__global__ void __launch_bounds__(NT) k_step_apply(SearchArgs A, const int64_t *key_in)
{
    __shared__ int64_t s_key;
    if (A.fs[FS_DONE]) return;
    const int64_t t = A.fs[FS_T] + 1;
    if (threadIdx.x == 0) s_key = *key_in;
    __syncthreads();
    const int64_t key = s_key;
    if (key == KEY_NONE || t > A.iters) {
        if (threadIdx.x == 0) { A.fs[FS_DONE] = 1; if (key == KEY_NONE) A.fs[FS_ERR] = 2; }
        return;
    }
    const uint32_t r = (uint32_t)(key & 0xffffffffu);
    const int64_t f = key >> 32;
    int a, b, c;
    unrank<K>(r, A.I.n, A.M, a, b, c);
    for (int j = threadIdx.x; j < A.I.m; j += NT) {
        const uint32_t *ar = A.I.Arow + (size_t)j * A.I.NWn;
        int d = (((__ldg(ar + (a >> 5)) ^ A.vb[a >> 5]) >> (a & 31)) & 1u) ? -1 : 1;
        if (K >= 2) d += (((__ldg(ar + (b >> 5)) ^ A.vb[b >> 5]) >> (b & 31)) & 1u) ? -1 : 1;
        if (K == 3) d += (((__ldg(ar + (c >> 5)) ^ A.vb[c >> 5]) >> (c & 31)) & 1u) ? -1 : 1;
        A.Y[j] -= 2 * d;
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        A.vb[a >> 5] ^= 1u << (a & 31);
        if (K >= 2) A.vb[b >> 5] ^= 1u << (b & 31);
        if (K == 3) A.vb[c >> 5] ^= 1u << (c & 31);
        if (A.L > 0) {
            const int64_t R1 = A.L + 1;
            if (t > A.L) {
                uint32_t old = A.ring[(t - A.L) % R1];
                if (old >= A.lo && old < A.hi) A.tabu[old >> 5] &= ~(1u << (old & 31));
            }
            if (r >= A.lo && r < A.hi) A.tabu[r >> 5] |= 1u << (r & 31);
            A.ring[t % R1] = r;
        }
        if (A.trace_r) A.trace_r[t - 1] = r;
        if (A.trace_f) A.trace_f[t - 1] = f;
        A.fs[FS_F] = f; A.fs[FS_T] = t;
        if (f < A.fs[FS_BEST]) { A.fs[FS_BEST] = f; A.fs[FS_BESTIT] = t; }
        if (f == 0 && A.fs[FS_ZERO] < 0) A.fs[FS_ZERO] = t;
        if ((A.stop_on_zero && f == 0) || t >= A.iters) A.fs[FS_DONE] = 1;
    }
}

// Debug: dump the plan of the current state (one CTA): [vmin, Upad, base, H[0..n], seg[0..Upad], bins.x, bins.y]
template <int K>
__global__ void __launch_bounds__(NT, 1) k_debug_plan(SearchArgs A, int32_t *out)
{
    extern __shared__ __align__(16) unsigned char sm[];
    __shared__ PlanScalars ps;
    const Smem L = smem_layout(A.I.m, A.I.n, A.I.W, A.I.NWn, K);
    load_state(A, sm, L);
    build_plan<K>(A.I, sm, L, ps);
    if (threadIdx.x == 0) {
        const int *Hs = (const int *)(sm + L.H);
        const int *seg = (const int *)(sm + L.seg);
        const int2 *bins = (const int2 *)(sm + L.bins);
        int o = 0;
        out[o++] = ps.vmin; out[o++] = ps.Upad; out[o++] = ps.base;
        for (int b = 0; b <= A.I.n; b++) out[o++] = Hs[b];
        for (int u = 0; u <= ps.Upad; u++) out[o++] = seg[u];
        for (int q = 0; q < ps.Upad + 2 * K; q++) { out[o++] = bins[q].x; out[o++] = bins[q].y; }
    }
}

template <int K>
__global__ void k_unrank(int n, uint32_t M, const int64_t *ranks, int64_t count, int32_t *out, int32_t *bad)
{
    for (int64_t q = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; q < count; q += (int64_t)gridDim.x * blockDim.x) {
        int64_t r = ranks[q];
        if (r < 0 || r >= (int64_t)M) { *bad = 1; out[3 * q] = out[3 * q + 1] = out[3 * q + 2] = -1; continue; }
        int a, b, c;
        unrank<K>((uint32_t)r, n, M, a, b, c);
        out[3 * q] = a; out[3 * q + 1] = b; out[3 * q + 2] = c;
    }
}

__global__ void k_fill_i64(int64_t *p, int64_t v, int64_t cnt)
{
    for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < cnt; i += (int64_t)gridDim.x * blockDim.x) p[i] = v;
}

}  // namespace

// ==========================================================================================
// Host side
// ==========================================================================================
typedef int (*nccl_allreduce_fn)(const void *, void *, size_t, int, int, void *, cudaStream_t);

struct lns_ctx {
    int device = 0;
    int m = 0, n = 0, W = 0, NWn = 0;
    uint32_t *d_Arow = nullptr;
    int32_t *d_H = nullptr;
    int numSMs = 0, smemOptin = 0;
    int part = 0, nparts = 1;
    void *comm = nullptr;
    nccl_allreduce_fn nccl_allreduce = nullptr;
    int blocks_override = 0;
    // run state
    uint32_t *d_vb = nullptr;
    int32_t *d_Y = nullptr;
    int64_t *d_fs = nullptr;
    int64_t *d_keys = nullptr;  // 3 persistent slots + 1 stepped accumulator + 1 eval output
    unsigned *d_bar = nullptr;  // [0..1] grid barrier, [2] stepped counter
    int8_t *d_V = nullptr;
    int32_t *d_Yin = nullptr;
    uint32_t *d_tabu = nullptr; size_t tabu_cap = 0;
    uint32_t *d_ring = nullptr; size_t ring_cap = 0;
    int64_t *d_tr = nullptr, *d_tf = nullptr; size_t trace_cap = 0, trace_cap_f = 0;
    int32_t *d_fit = nullptr; size_t fit_cap = 0;
    cudaEvent_t ev0 = nullptr, ev1 = nullptr;
    double last_ms = 0.0;
    // stepped search
    bool step_active = false;
    int step_K = 0; int64_t step_iters = 0, step_L = 0; int step_flags = 0;
};

namespace {

struct DeviceGuard {
    int prev = -1;
    explicit DeviceGuard(int dev) { cudaGetDevice(&prev); if (prev != dev) cudaSetDevice(dev); }
    ~DeviceGuard() { int cur; cudaGetDevice(&cur); if (prev >= 0 && cur != prev) cudaSetDevice(prev); }
};

lns_status fail(lns_status st, const std::string &msg) { g_err = msg; return st; }

#define CK(call)                                                                                   \
    do {                                                                                           \
        cudaError_t _e = (call);                                                                   \
        if (_e != cudaSuccess) return fail(LNS_ECUDA, std::string(#call) + ": " + cudaGetErrorString(_e)); \
    } while (0)

int64_t comb_k(int64_t n, int k)
{
    if (k == 1) return n;
    if (k == 2) return n * (n - 1) / 2;
    if (k == 3) return n * (n - 1) * (n - 2) / 6;
    return -1;
}

DevInst dev_inst(const lns_ctx *c) { return DevInst{c->m, c->n, c->W, c->NWn, c->d_Arow, c->d_H}; }

template <typename T>
lns_status grow(T *&p, size_t &cap, size_t need)
{
    if (need <= cap && p) return LNS_OK;
    if (p) cudaFree(p);
    p = nullptr; cap = 0;
    if (cudaMalloc(&p, need * sizeof(T) + 16) != cudaSuccess) { cudaGetLastError(); return fail(LNS_ENOMEM, "cudaMalloc failed"); }
    cap = need;
    return LNS_OK;
}

uint64_t splitmix64_next(uint64_t &s)
{
    s += 0x9E3779B97F4A7C15ULL;
    uint64_t z = s;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ULL;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBULL;
    return z ^ (z >> 31);
}

void vector_from_seed(int n, uint64_t seed, int8_t *V)
{
    uint64_t s = seed, w = 0;
    for (int i = 0; i < n; i++) {
        if (i % 64 == 0) w = splitmix64_next(s);
        V[i] = ((w >> (i % 64)) & 1) ? -1 : 1;
    }
}

void slice_of(uint32_t M, int part, int nparts, uint32_t &lo, uint32_t &hi)
{
    auto B = [&](int g) -> uint32_t {
        if (g >= nparts) return M;
        return 32u * (uint32_t)(((uint64_t)M * g / nparts) / 32);
    };
    lo = B(part);
    hi = B(part + 1);
}

template <int K>
void set_smem_attr(size_t bytes)
{
    cudaFuncSetAttribute(k_search<K>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)bytes);
    cudaFuncSetAttribute(k_step_eval<K, false>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)bytes);
    cudaFuncSetAttribute(k_step_eval<K, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)bytes);
}

lns_status check_k(const lns_ctx *c, int k, uint32_t &M, size_t &smem)
{
    if (!c) return fail(LNS_EINVAL, "null context");
    if (k < 1 || k > 3) return fail(LNS_EINVAL, "k must be 1, 2 or 3");
    if (c->n < k) return fail(LNS_EINVAL, "n < k");
    int64_t Mk = comb_k(c->n, k);
    if (Mk >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "C(n,k) >= 2^32-1");
    M = (uint32_t)Mk;
    Smem L = smem_layout(c->m, c->n, c->W, c->NWn, k);
    smem = (size_t)L.total;
    if ((int)smem > c->smemOptin - (int)sizeof(PlanScalars) - 64) return fail(LNS_ERANGE, "bit-packed A does not fit in shared memory");
    return LNS_OK;
}

// Blocks per search for the persistent kernel.
int search_blocks(const lns_ctx *c, uint32_t span, int occ)
{
    int cap = c->numSMs * occ;
    if (c->blocks_override > 0) return std::min(c->blocks_override, cap);
    int nb = (int)std::min<int64_t>((int64_t)cap, std::max<int64_t>(1, span / 1024));
    return std::max(1, nb);
}

SearchArgs make_args(lns_ctx *c, uint32_t M, int64_t iters, int64_t L, int flags)
{
    SearchArgs A;
    A.I = dev_inst(c);
    A.M = M;
    slice_of(M, c->part, c->nparts, A.lo, A.hi);
    A.iters = iters; A.L = L; A.stop_on_zero = (flags & LNS_STOP_ON_ZERO) ? 1 : 0;
    A.vb = c->d_vb; A.Y = c->d_Y; A.fs = c->d_fs; A.tabu = c->d_tabu; A.ring = c->d_ring;
    A.keys = c->d_keys; A.bar = c->d_bar; A.trace_r = c->d_tr; A.trace_f = c->d_tf;
    return A;
}

// Prepare a search: V0 -> state, tabu/ring/trace buffers cleared.
lns_status search_setup(lns_ctx *c, int k, uint32_t M, int64_t iters, int64_t L, uint64_t seed,
                        const int8_t *V0, cudaStream_t st)
{
    lns_status s;
    std::vector<int8_t> hv;
    if (V0) CK(cudaMemcpyAsync(c->d_V, V0, c->n, cudaMemcpyDefault, st));
    else {
        hv.resize(c->n);
        vector_from_seed(c->n, seed, hv.data());
        CK(cudaMemcpyAsync(c->d_V, hv.data(), c->n, cudaMemcpyHostToDevice, st));
    }
    size_t tw = (M + 31) / 32;
    if ((s = grow(c->d_tabu, c->tabu_cap, tw)) != LNS_OK) return s;
    CK(cudaMemsetAsync(c->d_tabu, 0, tw * 4, st));
    if (L > 0) {
        if ((s = grow(c->d_ring, c->ring_cap, (size_t)L + 1)) != LNS_OK) return s;
    }
    size_t tc = (size_t)std::max<int64_t>(iters, 1);
    if ((s = grow(c->d_tr, c->trace_cap, tc)) != LNS_OK) return s;
    if ((s = grow(c->d_tf, c->trace_cap_f, tc)) != LNS_OK) return s;
    k_fill_i64<<<1, 32, 0, st>>>(c->d_keys, KEY_NONE, 5);
    CK(cudaMemsetAsync(c->d_bar, 0, 4 * sizeof(unsigned), st));
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, nullptr, c->d_fs);
    CK(cudaGetLastError());
    (void)k;
    return LNS_OK;
}

lns_status search_finish(lns_ctx *c, int64_t iters, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit,
                         lns_result *res, cudaStream_t st)
{
    int64_t fs[FS_N];
    CK(cudaMemcpyAsync(fs, c->d_fs, sizeof(fs), cudaMemcpyDeviceToHost, st));
    std::vector<uint32_t> vb(c->NWn);
    CK(cudaMemcpyAsync(vb.data(), c->d_vb, 4 * c->NWn, cudaMemcpyDeviceToHost, st));
    CK(cudaStreamSynchronize(st));
    if (fs[FS_ERR] == 1) return fail(LNS_EINVAL, "V0 entries must be +1 or -1");
    if (fs[FS_ERR] == 2) return fail(LNS_ENOADMISSIBLE, "no admissible move");
    int64_t done = fs[FS_T];
    if (trace_rank && done > 0) CK(cudaMemcpyAsync(trace_rank, c->d_tr, done * 8, cudaMemcpyDefault, st));
    if (trace_fit && done > 0) CK(cudaMemcpyAsync(trace_fit, c->d_tf, done * 8, cudaMemcpyDefault, st));
    if (V_out) {
        std::vector<int8_t> hv(c->n);
        for (int i = 0; i < c->n; i++) hv[i] = ((vb[i / 32] >> (i % 32)) & 1) ? -1 : 1;
        CK(cudaMemcpyAsync(V_out, hv.data(), c->n, cudaMemcpyDefault, st));
    }
    CK(cudaStreamSynchronize(st));
    (void)iters;
    if (res) {
        res->iters_done = done; res->final_f = fs[FS_F]; res->best_f = fs[FS_BEST];
        res->best_iter = fs[FS_BESTIT]; res->first_zero_iter = fs[FS_ZERO];
        res->solved = fs[FS_BEST] == 0; res->reserved = 0;
    }
    return LNS_OK;
}

template <int K>
lns_status launch_search(lns_ctx *c, const SearchArgs &A, size_t smem, cudaStream_t st)
{
    set_smem_attr<K>(smem);
    int occ = 0;
    CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k_search<K>, NT, smem));
    if (occ < 1) return fail(LNS_ERANGE, "persistent kernel does not fit on an SM");
    int nb = search_blocks(c, A.hi - A.lo, occ);
    SearchArgs a = A;
    void *args[] = {&a};
    CK(cudaEventRecord(c->ev0, st));
    CK(cudaLaunchCooperativeKernel((void *)k_search<K>, dim3(nb), dim3(NT), args, smem, st));
    CK(cudaEventRecord(c->ev1, st));
    return LNS_OK;
}

template <int K>
lns_status launch_step_eval(lns_ctx *c, const SearchArgs &A, size_t smem, int64_t *key_out, int32_t *fit_out,
                            bool all, cudaStream_t st)
{
    set_smem_attr<K>(smem);
    int occ = 0;
    CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k_step_eval<K, false>, NT, smem));
    if (occ < 1) return fail(LNS_ERANGE, "eval kernel does not fit on an SM");
    SearchArgs a = A;
    a.keys = c->d_keys + 3;
    a.bar = c->d_bar + 2;
    int nb = search_blocks(c, A.hi - A.lo, occ);
    if (all) {
        nb = (int)std::min<int64_t>(std::max<int64_t>(1, (A.hi - A.lo) / 1024), 4LL * c->numSMs * occ);
        k_step_eval<K, true><<<nb, NT, smem, st>>>(a, key_out, fit_out);
    } else {
        k_step_eval<K, false><<<nb, NT, smem, st>>>(a, key_out, fit_out);
    }
    CK(cudaGetLastError());
    return LNS_OK;
}

template <int K>
lns_status launch_step_apply(const SearchArgs &A, const int64_t *key, cudaStream_t st)
{
    k_step_apply<K><<<1, NT, 0, st>>>(A, key);
    CK(cudaGetLastError());
    return LNS_OK;
}

lns_status dispatch_search(lns_ctx *c, int k, const SearchArgs &A, size_t smem, cudaStream_t st)
{
    switch (k) {
    case 1: return launch_search<1>(c, A, smem, st);
    case 2: return launch_search<2>(c, A, smem, st);
    default: return launch_search<3>(c, A, smem, st);
    }
}
lns_status dispatch_step_eval(lns_ctx *c, int k, const SearchArgs &A, size_t smem, int64_t *key_out,
                              int32_t *fit_out, bool all, cudaStream_t st)
{
    switch (k) {
    case 1: return launch_step_eval<1>(c, A, smem, key_out, fit_out, all, st);
    case 2: return launch_step_eval<2>(c, A, smem, key_out, fit_out, all, st);
    default: return launch_step_eval<3>(c, A, smem, key_out, fit_out, all, st);
    }
}
lns_status dispatch_step_apply(int k, const SearchArgs &A, const int64_t *key, cudaStream_t st)
{
    switch (k) {
    case 1: return launch_step_apply<1>(A, key, st);
    case 2: return launch_step_apply<2>(A, key, st);
    default: return launch_step_apply<3>(A, key, st);
    }
}

lns_status resolve_tenure(int64_t M, int64_t tenure, int64_t &L)
{
    L = tenure < 0 ? M / 6 : tenure;
    if (L >= M) return fail(LNS_ERANGE, "tenure >= C(n,k): no admissible move would remain");
    return LNS_OK;
}

}  // namespace

// ==========================================================================================
// C ABI
// ==========================================================================================
extern "C" {

const char *lns_strerror(lns_status s)
{
    switch (s) {
    case LNS_OK: return "ok";
    case LNS_EINVAL: return "invalid argument";
    case LNS_ERANGE: return "size limit exceeded";
    case LNS_ENOMEM: return "out of memory";
    case LNS_ECUDA: return "CUDA error";
    case LNS_ENCCL: return "NCCL error";
    case LNS_ENOADMISSIBLE: return "no admissible neighbour";
    default: return "unknown status";
    }
}

const char *lns_last_error(void) { return g_err.c_str(); }
int32_t lns_version(void) { return LNS_VERSION_NUM; }
int64_t lns_neighborhood_size(int32_t n, int32_t k)
{
    if (k < 1 || k > 3) return -1;
    return n < k ? 0 : comb_k(n, k);
}

lns_status lns_create(const int8_t *A, int32_t m, int32_t n, const int32_t *S, int32_t device, lns_ctx **out)
{
    if (!out || !A || !S) return fail(LNS_EINVAL, "null argument");
    *out = nullptr;
    if (m < 1 || n < 1) return fail(LNS_EINVAL, "m and n must be >= 1");
    if (60LL * m * n + 2LL * m >= (int64_t)INT32_MAX) return fail(LNS_ERANGE, "60 m n + 2 m >= 2^31");
    if (n > 4096) return fail(LNS_ERANGE, "n > 4096");
    int ndev = 0;
    CK(cudaGetDeviceCount(&ndev));
    if (device < 0 || device >= ndev) return fail(LNS_EINVAL, "bad device index");
    DeviceGuard g(device);
    std::vector<int8_t> hA((size_t)m * n);
    std::vector<int32_t> hS(m);
    CK(cudaMemcpy(hA.data(), A, hA.size(), cudaMemcpyDefault));
    CK(cudaMemcpy(hS.data(), S, 4 * (size_t)m, cudaMemcpyDefault));
    const int NWn = (n + 31) / 32, W = (m + 31) / 32;
    std::vector<uint32_t> arow((size_t)m * NWn, 0u);
    std::vector<int32_t> H(n + 1, 0);
    for (int j = 0; j < m; j++) {
        for (int i = 0; i < n; i++) {
            int8_t a = hA[(size_t)j * n + i];
            if (a != 1 && a != -1) return fail(LNS_EINVAL, "A entries must be +1 or -1");
            if (a < 0) arow[(size_t)j * NWn + i / 32] |= 1u << (i % 32);
        }
        if (hS[j] < 0 || hS[j] > n) return fail(LNS_EINVAL, "S entries must lie in [0, n]");
        H[hS[j]]++;
    }
    lns_ctx *c = new lns_ctx();
    c->device = device; c->m = m; c->n = n; c->W = W; c->NWn = NWn;
    auto cleanup = [&](lns_status s) { lns_destroy(c); return s; };
    if (cudaDeviceGetAttribute(&c->numSMs, cudaDevAttrMultiProcessorCount, device) != cudaSuccess ||
        cudaDeviceGetAttribute(&c->smemOptin, cudaDevAttrMaxSharedMemoryPerBlockOptin, device) != cudaSuccess)
        return cleanup(fail(LNS_ECUDA, "device attributes"));
    if (cudaMalloc(&c->d_Arow, arow.size() * 4) != cudaSuccess || cudaMalloc(&c->d_H, (n + 1) * 4) != cudaSuccess ||
        cudaMalloc(&c->d_vb, NWn * 4) != cudaSuccess || cudaMalloc(&c->d_Y, m * 4) != cudaSuccess ||
        cudaMalloc(&c->d_fs, FS_N * 8) != cudaSuccess || cudaMalloc(&c->d_keys, 8 * 8) != cudaSuccess ||
        cudaMalloc(&c->d_bar, 4 * sizeof(unsigned)) != cudaSuccess || cudaMalloc(&c->d_V, n) != cudaSuccess ||
        cudaMalloc(&c->d_Yin, m * 4) != cudaSuccess) {
        cudaGetLastError();
        return cleanup(fail(LNS_ENOMEM, "cudaMalloc failed"));
    }
    if (cudaMemcpy(c->d_Arow, arow.data(), arow.size() * 4, cudaMemcpyHostToDevice) != cudaSuccess ||
        cudaMemcpy(c->d_H, H.data(), (n + 1) * 4, cudaMemcpyHostToDevice) != cudaSuccess ||
        cudaMemset(c->d_bar, 0, 4 * sizeof(unsigned)) != cudaSuccess ||
        cudaEventCreate(&c->ev0) != cudaSuccess || cudaEventCreate(&c->ev1) != cudaSuccess)
        return cleanup(fail(LNS_ECUDA, "upload"));
    *out = c;
    return LNS_OK;
}

void lns_destroy(lns_ctx *c)
{
    if (!c) return;
    DeviceGuard g(c->device);
    cudaFree(c->d_Arow); cudaFree(c->d_H); cudaFree(c->d_vb); cudaFree(c->d_Y); cudaFree(c->d_fs);
    cudaFree(c->d_keys); cudaFree(c->d_bar); cudaFree(c->d_V); cudaFree(c->d_Yin); cudaFree(c->d_tabu);
    cudaFree(c->d_ring); cudaFree(c->d_tr); cudaFree(c->d_tf); cudaFree(c->d_fit);
    if (c->ev0) cudaEventDestroy(c->ev0);
    if (c->ev1) cudaEventDestroy(c->ev1);
    delete c;
}

lns_status lns_config(lns_ctx *c, int32_t blocks)
{
    if (!c || blocks < 0) return fail(LNS_EINVAL, "bad config");
    c->blocks_override = blocks;
    return LNS_OK;
}

double lns_last_kernel_ms(lns_ctx *c) { return c ? c->last_ms : 0.0; }

lns_status lns_set_partition(lns_ctx *c, int32_t part, int32_t nparts)
{
    if (!c || nparts < 1 || part < 0 || part >= nparts) return fail(LNS_EINVAL, "bad partition");
    c->part = part; c->nparts = nparts;
    return LNS_OK;
}

lns_status lns_attach_comm(lns_ctx *c, void *comm, int32_t rank, int32_t world)
{
    if (!c) return fail(LNS_EINVAL, "null context");
    if (!comm) { c->comm = nullptr; c->part = 0; c->nparts = 1; return LNS_OK; }
    if (world < 1 || rank < 0 || rank >= world) return fail(LNS_EINVAL, "bad rank/world");
    void *h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_NOLOAD);
    if (!h) h = dlopen("libnccl.so.2", RTLD_NOW);
    void *sym = h ? dlsym(h, "ncclAllReduce") : dlsym(RTLD_DEFAULT, "ncclAllReduce");
    if (!sym) return fail(LNS_ENCCL, "ncclAllReduce not found (load torch's libnccl first)");
    c->nccl_allreduce = (nccl_allreduce_fn)sym;
    c->comm = comm;
    c->part = rank; c->nparts = world;
    return LNS_OK;
}

lns_status lns_eval_neighborhood(lns_ctx *c, int32_t k, const int8_t *V, const int32_t *Y, const uint32_t *tabu_bits,
                                 int64_t *best_fitness, int64_t *best_rank, void *stream)
{
    uint32_t M; size_t smem;
    lns_status s = check_k(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (!V || !Y || !best_fitness || !best_rank) return fail(LNS_EINVAL, "null argument");
    DeviceGuard g(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    size_t tw = (M + 31) / 32;
    if ((s = grow(c->d_tabu, c->tabu_cap, tw)) != LNS_OK) return s;
    if (tabu_bits) CK(cudaMemcpyAsync(c->d_tabu, tabu_bits, tw * 4, cudaMemcpyDefault, st));
    else CK(cudaMemsetAsync(c->d_tabu, 0, tw * 4, st));
    CK(cudaMemcpyAsync(c->d_V, V, c->n, cudaMemcpyDefault, st));
    CK(cudaMemcpyAsync(c->d_Yin, Y, 4 * (size_t)c->m, cudaMemcpyDefault, st));
    k_fill_i64<<<1, 32, 0, st>>>(c->d_keys, KEY_NONE, 5);
    CK(cudaMemsetAsync(c->d_bar, 0, 4 * sizeof(unsigned), st));
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, c->d_Yin, c->d_fs);
    CK(cudaGetLastError());
    SearchArgs A = make_args(c, M, 1, 0, 0);
    CK(cudaEventRecord(c->ev0, st));
    if ((s = dispatch_step_eval(c, k, A, smem, c->d_keys + 4, nullptr, false, st)) != LNS_OK) return s;
    CK(cudaEventRecord(c->ev1, st));
    int64_t key, fs[FS_N];
    CK(cudaMemcpyAsync(&key, c->d_keys + 4, 8, cudaMemcpyDeviceToHost, st));
    CK(cudaMemcpyAsync(fs, c->d_fs, sizeof(fs), cudaMemcpyDeviceToHost, st));
    CK(cudaStreamSynchronize(st));
    float ms = 0; cudaEventElapsedTime(&ms, c->ev0, c->ev1); c->last_ms = ms;
    if (fs[FS_ERR]) return fail(LNS_EINVAL, "V must be +-1 and Y must equal A V");
    if (key == KEY_NONE) { *best_fitness = -1; *best_rank = -1; return fail(LNS_ENOADMISSIBLE, "all ranks tabu"); }
    *best_fitness = key >> 32;
    *best_rank = key & 0xffffffffLL;
    return LNS_OK;
}

lns_status lns_eval_all(lns_ctx *c, int32_t k, const int8_t *V, int32_t *fitness_out, void *stream)
{
    uint32_t M; size_t smem;
    lns_status s = check_k(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (!V || !fitness_out) return fail(LNS_EINVAL, "null argument");
    DeviceGuard g(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    if ((s = grow(c->d_fit, c->fit_cap, M)) != LNS_OK) return s;
    size_t tw = (M + 31) / 32;
    if ((s = grow(c->d_tabu, c->tabu_cap, tw)) != LNS_OK) return s;
    CK(cudaMemsetAsync(c->d_tabu, 0, tw * 4, st));
    CK(cudaMemcpyAsync(c->d_V, V, c->n, cudaMemcpyDefault, st));
    k_fill_i64<<<1, 32, 0, st>>>(c->d_keys, KEY_NONE, 5);
    CK(cudaMemsetAsync(c->d_bar, 0, 4 * sizeof(unsigned), st));
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, nullptr, c->d_fs);
    SearchArgs A = make_args(c, M, 1, 0, 0);
    A.lo = 0; A.hi = M;
    CK(cudaEventRecord(c->ev0, st));
    if ((s = dispatch_step_eval(c, k, A, smem, c->d_keys + 4, c->d_fit, true, st)) != LNS_OK) return s;
    CK(cudaEventRecord(c->ev1, st));
    int64_t fs[FS_N];
    CK(cudaMemcpyAsync(fs, c->d_fs, sizeof(fs), cudaMemcpyDeviceToHost, st));
    CK(cudaMemcpyAsync(fitness_out, c->d_fit, 4 * (size_t)M, cudaMemcpyDefault, st));
    CK(cudaStreamSynchronize(st));
    float ms = 0; cudaEventElapsedTime(&ms, c->ev0, c->ev1); c->last_ms = ms;
    if (fs[FS_ERR]) return fail(LNS_EINVAL, "V must be +-1");
    return LNS_OK;
}

lns_status lns_step_begin(lns_ctx *c, int32_t k, int64_t max_iters, int64_t tenure, uint64_t seed, const int8_t *V0,
                          int32_t flags, void *stream)
{
    uint32_t M; size_t smem;
    lns_status s = check_k(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (max_iters < 0) return fail(LNS_EINVAL, "iters < 0");
    int64_t L;
    if ((s = resolve_tenure(M, tenure, L)) != LNS_OK) return s;
    DeviceGuard g(c->device);
    if ((s = search_setup(c, k, M, max_iters, L, seed, V0, (cudaStream_t)stream)) != LNS_OK) return s;
    c->step_active = true; c->step_K = k; c->step_iters = max_iters; c->step_L = L; c->step_flags = flags;
    return LNS_OK;
}

lns_status lns_step_eval(lns_ctx *c, int64_t *key_dev, void *stream)
{
    if (!c || !c->step_active || !key_dev) return fail(LNS_EINVAL, "no active stepped search");
    uint32_t M; size_t smem;
    lns_status s = check_k(c, c->step_K, M, smem);
    if (s != LNS_OK) return s;
    DeviceGuard g(c->device);
    SearchArgs A = make_args(c, M, c->step_iters, c->step_L, c->step_flags);
    return dispatch_step_eval(c, c->step_K, A, smem, key_dev, nullptr, false, (cudaStream_t)stream);
}

lns_status lns_step_apply(lns_ctx *c, const int64_t *key_dev, void *stream)
{
    if (!c || !c->step_active || !key_dev) return fail(LNS_EINVAL, "no active stepped search");
    uint32_t M; size_t smem;
    lns_status s = check_k(c, c->step_K, M, smem);
    if (s != LNS_OK) return s;
    DeviceGuard g(c->device);
    SearchArgs A = make_args(c, M, c->step_iters, c->step_L, c->step_flags);
    return dispatch_step_apply(c->step_K, A, key_dev, (cudaStream_t)stream);
}

lns_status lns_step_end(lns_ctx *c, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit, lns_result *res, void *stream)
{
    if (!c || !c->step_active) return fail(LNS_EINVAL, "no active stepped search");
    DeviceGuard g(c->device);
    c->step_active = false;
    return search_finish(c, c->step_iters, V_out, trace_rank, trace_fit, res, (cudaStream_t)stream);
}

lns_status lns_tabu_run(lns_ctx *c, int32_t k, int64_t iters, int64_t tenure, uint64_t seed, const int8_t *V0,
                        int32_t flags, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit, lns_result *res,
                        void *stream)
{
    uint32_t M; size_t smem;
    lns_status s = check_k(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (!res) return fail(LNS_EINVAL, "res is required");
    if (iters < 0) return fail(LNS_EINVAL, "iters < 0");
    int64_t L;
    if ((s = resolve_tenure(M, tenure, L)) != LNS_OK) return s;
    DeviceGuard g(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    if ((s = search_setup(c, k, M, iters, L, seed, V0, st)) != LNS_OK) return s;
    SearchArgs A = make_args(c, M, iters, L, flags);
    const bool stepped = c->comm != nullptr || c->nparts > 1 || (flags & LNS_FORCE_STEPPED);
    if (!stepped) {
        if (iters > 0 && (s = dispatch_search(c, k, A, smem, st)) != LNS_OK) return s;
    } else {
        if (c->nparts > 1 && !c->comm) return fail(LNS_EINVAL, "partitioned run needs a communicator (or use the stepped API)");
        int64_t *kb = c->d_keys + 4;
        CK(cudaEventRecord(c->ev0, st));
        for (int64_t t = 0; t < iters; t++) {
            if ((s = dispatch_step_eval(c, k, A, smem, kb, nullptr, false, st)) != LNS_OK) return s;
            if (c->comm) {
                int rc = c->nccl_allreduce(kb, kb, 1, /*ncclUint64*/ 5, /*ncclMin*/ 3, c->comm, st);
                if (rc != 0) return fail(LNS_ENCCL, "ncclAllReduce failed");
            }
            if ((s = dispatch_step_apply(k, A, kb, st)) != LNS_OK) return s;
            if ((flags & LNS_STOP_ON_ZERO) && (t % 64) == 63) {
                int64_t done;
                CK(cudaMemcpyAsync(&done, c->d_fs + FS_DONE, 8, cudaMemcpyDeviceToHost, st));
                CK(cudaStreamSynchronize(st));
                if (done) break;
            }
        }
        CK(cudaEventRecord(c->ev1, st));
    }
    s = search_finish(c, iters, V_out, trace_rank, trace_fit, res, st);
    float ms = 0;
    if (iters > 0 && cudaEventElapsedTime(&ms, c->ev0, c->ev1) == cudaSuccess) c->last_ms = ms;
    cudaGetLastError();
    return s;
}

lns_status lns_tabu_run_batch(lns_ctx *c, int32_t k, int32_t R, int64_t iters, int64_t tenure, uint64_t seed,
                              const int8_t *V0, int32_t flags, int8_t *V_out, lns_result *res, void *stream)
{
    if (!c || !res || R < 0) return fail(LNS_EINVAL, "bad argument");
    int savep = c->part, saven = c->nparts;
    void *savec = c->comm;
    c->part = 0; c->nparts = 1; c->comm = nullptr;
    lns_status s = LNS_OK;
    double total_ms = 0;
    for (int r = 0; r < R && s == LNS_OK; r++) {
        uint64_t st = seed + (uint64_t)r;
        uint64_t seed_r = splitmix64_next(st);
        const int8_t *v0 = V0 ? V0 + (size_t)r * c->n : nullptr;
        int8_t *vo = V_out ? V_out + (size_t)r * c->n : nullptr;
        s = lns_tabu_run(c, k, iters, tenure, seed_r, v0, flags & ~LNS_FORCE_STEPPED, vo, nullptr, nullptr, &res[r], stream);
        total_ms += c->last_ms;
    }
    c->last_ms = total_ms;
    c->part = savep; c->nparts = saven; c->comm = savec;
    return s;
}

// Undocumented debug export (tests/tools only): plan of V for neighbourhood k, see k_debug_plan.
lns_status lns_debug_plan(lns_ctx *c, int32_t k, const int8_t *V, int32_t *out_host, int64_t cap)
{
    uint32_t M; size_t smem;
    lns_status s = check_k(c, k, M, smem);
    if (s != LNS_OK) return s;
    DeviceGuard g(c->device);
    int32_t *d_out = nullptr;
    CK(cudaMalloc(&d_out, cap * 4));
    CK(cudaMemcpy(c->d_V, V, c->n, cudaMemcpyDefault));
    k_init<<<1, NT>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, nullptr, c->d_fs);
    SearchArgs A = make_args(c, M, 1, 0, 0);
    if (k == 1) { cudaFuncSetAttribute(k_debug_plan<1>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem); k_debug_plan<1><<<1, NT, smem>>>(A, d_out); }
    else if (k == 2) { cudaFuncSetAttribute(k_debug_plan<2>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem); k_debug_plan<2><<<1, NT, smem>>>(A, d_out); }
    else { cudaFuncSetAttribute(k_debug_plan<3>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem); k_debug_plan<3><<<1, NT, smem>>>(A, d_out); }
    CK(cudaMemcpy(out_host, d_out, cap * 4, cudaMemcpyDeviceToHost));
    cudaFree(d_out);
    return LNS_OK;
}

lns_status lns_unrank(int32_t n, int32_t k, const int64_t *ranks, int64_t count, int32_t *out, void *stream)
{
    if (k < 1 || k > 3 || n < k) return fail(LNS_EINVAL, "bad n/k");
    if (count < 0 || (count > 0 && (!ranks || !out))) return fail(LNS_EINVAL, "bad buffers");
    int64_t Mk = comb_k(n, k);
    if (Mk >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "C(n,k) >= 2^32-1");
    if (count == 0) return LNS_OK;
    cudaStream_t st = (cudaStream_t)stream;
    int64_t *d_r = nullptr; int32_t *d_o = nullptr, *d_bad = nullptr;
    if (cudaMalloc(&d_r, count * 8) != cudaSuccess || cudaMalloc(&d_o, count * 12) != cudaSuccess ||
        cudaMalloc(&d_bad, 4) != cudaSuccess) {
        cudaFree(d_r); cudaFree(d_o); cudaGetLastError();
        return fail(LNS_ENOMEM, "cudaMalloc failed");
    }
    int bad = 0;
    cudaMemcpyAsync(d_r, ranks, count * 8, cudaMemcpyDefault, st);
    cudaMemsetAsync(d_bad, 0, 4, st);
    int blocks = (int)std::min<int64_t>((count + 255) / 256, 4096);
    if (k == 1) k_unrank<1><<<blocks, 256, 0, st>>>(n, (uint32_t)Mk, d_r, count, d_o, d_bad);
    else if (k == 2) k_unrank<2><<<blocks, 256, 0, st>>>(n, (uint32_t)Mk, d_r, count, d_o, d_bad);
    else k_unrank<3><<<blocks, 256, 0, st>>>(n, (uint32_t)Mk, d_r, count, d_o, d_bad);
    cudaMemcpyAsync(out, d_o, count * 12, cudaMemcpyDefault, st);
    cudaMemcpyAsync(&bad, d_bad, 4, cudaMemcpyDeviceToHost, st);
    cudaError_t e = cudaStreamSynchronize(st);
    cudaFree(d_r); cudaFree(d_o); cudaFree(d_bad);
    if (e != cudaSuccess) return fail(LNS_ECUDA, cudaGetErrorString(e));
    if (bad) return fail(LNS_EINVAL, "rank out of range");
    return LNS_OK;
}

}  // extern "C"

// lns.cu -- sm_100a kernels and C ABI (include/lns.h) of the k-Hamming tabu search on the
// Permuted Perceptron Problem (Luong, Melab, Talbi, LSPP@IPDPS 2010; PAPER.md).
//
// Design:
//  * A is bit-packed once (sign bits, bit = 1 <=> -1). Per iteration every CTA builds, in shared
//    memory, a "plan" of the current state: rows sorted by Y (counting sort over the lattice
//    Y = vmin + 2u), the sign bits x_jc = [A_jc V_c = -1] permuted into that row order and stored
//    [row-word][column], the pieces (segment x row-word) of equal-Y rows, and per-bin constants.
//  * A neighbour F = {a<b<c} moves row j to Y'_j = Y_j - 2k + 4 t_j, t_j = #{i in F : x_ji = 1}
//    (PAPER.md:227-229 with V' = V xor F). All rows of one Y-segment land in the same k+1 bins, so
//    the new histogram H' only needs, per segment, how many rows have t = 0..k.
//    Those counts come from bit-sliced t (LOP3) and POPC over the segment's row words; a shift
//    register over the segment lattice turns them into H'(b) and the fitness (60|b|-weighted
//    penalty on negative bins, |H - H'| on bins 0..n), exactly, in integers.
//  * Ranks are lexicographic (reading R6); each lane unranks exactly (integer combinatorial number
//    system, float estimate + integer correction). The (fitness, rank) pair is packed into one
//    63-bit key, so a u64 MIN gives "least fitness, lowest rank" (reading R5) at warp, CTA, grid and
//    (NCCL) multi-GPU level.
//  * The whole tabu search runs in ONE persistent cooperative kernel. Per iteration each CTA
//    publishes its best key into a parity-tagged slot and polls all slots (one exchange, no
//    separate barrier); every CTA applies the winning move to its own shared copy of (V, Y).
//    The tabu list is the literal until[] array of the oracle (rank r is tabu while
//    until[r] >= t), each CTA owning (and caching in shared memory) the slice it evaluates.
#include "lns.h"

#include <cuda_runtime.h>
#include <dlfcn.h>

#include <algorithm>
#include <climits>
#include <cstdlib>
#include <cmath>
#include <cstdio>
#include <cstring>
#include <ctime>
#include <string>
#include <map>
#include <mutex>
#include <vector>

#define LNS_VERSION_NUM 200

namespace {

constexpr int64_t KEY_NONE = INT64_MAX;
#ifndef LNS_NT
#define LNS_NT 1024
#endif
constexpr int NT = LNS_NT;  // threads per CTA
constexpr int NWARP = NT / 32;
constexpr unsigned FULL = 0xffffffffu;
constexpr int MAX_SLOTS = 1024;  // CTAs per search that can exchange keys

thread_local std::string g_err;

// Optional per-phase cycle accounting (compile with -DLNS_PHASE_TIMING; tools/profiling only).
#ifdef LNS_PHASE_TIMING
constexpr int NPH = 12;
__shared__ long long s_ph[NPH];
__shared__ long long s_last;
__device__ unsigned long long g_ph[NPH];
#define PH(i)                                                        \
    do {                                                             \
        if (threadIdx.x == 0) {                                      \
            const long long _now = clock64();                        \
            s_ph[i] += _now - s_last;                                \
            s_last = _now;                                           \
        }                                                            \
    } while (0)
#else
#define PH(i) do { } while (0)
#endif

// ------------------------------------------------------------------------------------------
// Device data
// ------------------------------------------------------------------------------------------
struct DevInst {
    int32_t m, n, W, NWn;  // W = ceil(m/32) row words, NWn = ceil(n/32) column words
    int32_t XW;            // row words X has room for: W, or 2W + 1 with padded placement
    int32_t pad;           // padded placement: no segment of <= 32 rows straddles a row word
    const uint32_t *Arow;  // m x NWn, bit (i%32) of word i/32 = 1 <=> A[j][i] = -1
    const int32_t *H;      // n+1 bins of S
    int32_t maxS;          // largest b with H_b > 0
    int32_t pkw;           // m > 255: the packed (byte-window) plan is tried per iteration
};

// fstate layout (int64): current f, iterations done, best f, best iter, first zero iter, done, error
enum { FS_F = 0, FS_T, FS_BEST, FS_BESTIT, FS_ZERO, FS_DONE, FS_ERR, FS_N };
// FS_ERR: 1 = bad V0, 2 = no admissible move, 3 = peer exchange timed out, 4 = grid exchange timed out
#define MAX_PEERS 16
#define LNS_MAXPH 4

struct SearchArgs {
    DevInst I;
    uint32_t M;             // C(n,k)
    uint32_t lo, hi;        // rank slice of this device
    int64_t iters;          // iterations to run (persistent) / capacity (stepped)
    int64_t L;              // tenure
    int32_t stop_on_zero;
    int32_t a_in_smem;      // stage A's bit rows in shared memory
    int32_t until_smem;     // cache the CTA's until[] slice in shared memory (1 = yes)
    int32_t tri_smem;       // cache the flip sets of the CTA's slice in shared memory (1 = yes)
    int32_t slice_cap;      // capacity (ranks) of the per-CTA shared caches
    int32_t aspiration;     // a tabu move is admissible when it beats the best fitness so far
    int32_t sol_list;       // LNS_TABU_SOLUTIONS (reading R3'): the tabu list holds visited solutions
    uint32_t *ring;         // sol_list: V_s in slot s mod L, L x NWn words per group (group gg at gg L NWn)
    uint32_t *Xg;          // non-null: X lives in global memory, XW * n words per CTA (large m x n)
    // batched restarts (lns_tabu_run_batch): the grid is split into `groups` groups of CTAs; group g
    // runs restarts g, g + groups, ... each from V0s[r] and writes res[r] / vouts[r]. R = 0: one
    // search from the state in (vb, Y, fs).
    int32_t groups, R;
    // batched schedule: phase q runs runs [phr0[q], phr0[q] + phR[q]) on phG[q] groups of phnb[q]
    // CTAs (group g takes runs phr0 + g, phr0 + g + phG, ...); phase groups have their own exchange
    // slots and until[] arrays (global group index phgb[q] + g), so no grid barrier separates phases
    int32_t nph;
    int32_t phG[LNS_MAXPH], phnb[LNS_MAXPH], phgb[LNS_MAXPH], phr0[LNS_MAXPH], phR[LNS_MAXPH];
    const int8_t *V0s;      // R x n
    int64_t *res;           // R x FS_N
    uint32_t *vouts;        // R x NWn
    uint32_t *vb;           // state: NWn words of V's sign bits
    int32_t *Y;             // state: m
    int64_t *fs;            // FS_N
    uint32_t *until;        // M entries: rank r is tabu at iteration t iff until[r] >= t
    // compact tabu state (bits_mode), used instead of a global until[] when the
    // CTA's slice does not fit in shared memory and neither variant (aspiration, solution list) is
    // on: bit r of tbits = rank r is in the FIFO of the last L accepted ranks; tring[(s-1) % L] = the
    // rank accepted at iteration s (only when the run can outlast the tenure: ring_on)
    uint32_t *tbits;        // per group: bit_words words
    uint32_t *tring;        // per group: L words (ring_on)
    int32_t bits_mode, ring_on;
    uint32_t bit_words;     // words per group bitmap (ceil(M/32))
    int64_t *slots;         // 3 x MAX_SLOTS parity-tagged keys (persistent) / accumulator (stepped)
    unsigned *counter;      // stepped: last-CTA counter
    int64_t *trace_r, *trace_f;
    // device-initiated multi-GPU exchange (lns_attach_peers): npeers > 0 = every CTA of
    // every partition meets in the exchange buffers peers[0..npeers), own buffer peers[part]
    unsigned long long *const *peers;
    int32_t npeers, part;
    int64_t nb_total;       // CTAs over all partitions (the arrival count per exchange)
    int64_t timeout_ns;     // a partition missing for this long ends the run (FS_ERR = 3)
    int64_t grid_timeout_ns;  // a CTA of this grid missing at an exchange for this long ends the run (FS_ERR = 4)
    int32_t plain_launch;   // LNS_PLAIN_LAUNCH: cudaLaunchKernel instead of the cooperative launch
    int32_t enc_keys;       // keys carry the flip set (enc_flip) instead of the rank: no unranking after the exchange
};

// The CTA's X (sorted sign bits): shared memory, or its own slot of the global fallback buffer.
#define X_OF(A, sm, L) ((A).Xg ? (A).Xg + (size_t)blockIdx.x * (A).I.XW * (A).I.n : (uint32_t *)((sm) + (L).X))

// Shared-memory carve-up (identical on host and device). The bit-packed A (Ar) and the until[]
// slice are staged only when they fit.
struct Smem {
    int X, Y, vb, H, cnt, seg, cur, pofs, rowAt, bins, pieces, pk, pstart, T2, T3, base_end, Ar, a_end;
};

__host__ __device__ inline int align16(int x) { return (x + 15) & ~15; }

// Bin counts fit a byte (the packed evaluation path, eval_fit_packed) when m <= 255.
#define PACKED_MAX_M 255
#ifndef PK_UNROLL
#define PK_UNROLL 1
#endif
constexpr int kPkUnroll = PK_UNROLL;  // unroll of the packed piece loop
// byte_perm selectors of the packed records: h = window byte 0 moved to byte 1 (a final piece), or
// an always-zero byte (byte 7 of the window, unused for K <= 3) for a piece that completes no bin
#define PK_SEL_FIN 0x7707u
#define PK_SEL_NONE 0x7777u
#ifndef PK_PAIR
#define PK_PAIR 1
#endif

// XW = row words of X (I.XW: W, or 2W + 1 with padded placement)
__host__ __device__ inline Smem smem_layout(int m, int n, int W, int NWn, int K, int a_in_smem, int x_global = 0,
                                            int pkw = 0)
{
    Smem s;
    int o = 0;
    s.X = o;      o = align16(o + (x_global ? 0 : 4 * W * n));  // X in global memory when it cannot fit
    s.Y = o;      o = align16(o + 4 * m);
    s.vb = o;     o = align16(o + 4 * NWn);
    s.H = o;      o = align16(o + 4 * (n + 1));
    s.cnt = o;    o = align16(o + 4 * (n + 2 + 2 * K));  // conservative lattice Uc <= n + 1 + 2K
    s.seg = o;    o = align16(o + 4 * (n + 2));          // seg[0..U], U <= n + 1
    s.cur = o;    o = align16(o + 4 * (n + 2 + 2 * K));
    s.pofs = o;   o = align16(o + 4 * (n + 2));
    s.rowAt = o;  o = align16(o + 4 * (m > 32 * W ? m : 32 * W));  // row slots (holes = -1 when padded)
    s.bins = o;   o = align16(o + 8 * (n + 1 + 2 * K));  // NB = U + 2K bins
    s.pieces = o; o = align16(o + 8 * (n + 2 + W));      // P <= U + W - 1 pieces (+1 prefetch pad)
    s.pk = o;     o = align16(o + ((m <= PACKED_MAX_M || pkw) ? 16 * (n + 2 + W) : 0));  // packed-path records
    s.pstart = o; o = align16(o + 4 * (W + 1));
    s.T2 = o;     o = align16(o + 4 * n);                // C(y,2), y < n (u32)
    s.T3 = o;     o = align16(o + 4 * n);                // C(z,3), z < n (u32: C(n,3) < 2^32)
    s.base_end = o;
    s.Ar = o;
    if (a_in_smem) o = align16(o + 4 * m * NWn);
    s.a_end = o;  // the until[] slice (if cached) follows
    return s;
}

struct PlanScalars {
    // packed path, per walk q (set at the end of build_plan_pk): pkwk[q] = (X row-word base: shared
    // byte address, or the word offset of the global X; first record address; end record address;
    // address of pstart[first word + 1]); pkwt[q] = (initial window, trailing H bytes, trailing
    // bin negative, last point)
    uint4 pkwk[2], pkwt[2];
    int vmin, U, NB, P, ufirst;
    int fpen, fhd;  // block_fitness accumulators
    // linear regions: lattice points u < uneg are "deep negative" (all k+1
    // destinations negative: cost linear, aggregated as cneg - 240 sum t over the first rneg sorted
    // rows); points u >= utop land only above max(S) (zero cost) and are skipped
    int uneg, utop, rneg, cneg;
    // packed path (abs form): sum of H_b over the walked bins
    int hwalk;
    int pkok;  // this plan is the packed one (always for m <= 255; per iteration for m > 255, §5.11)
    int Wp;    // row words X holds this plan (ceil(row slots / 32); padded slots are holes)
    int rtop;  // rows below the top cut (points < utop), unpadded
    int vlo, Uc;  // conservative lattice of the NEXT plan: every Y lies in vlo + 2 [0, Uc)
    // packed path, parity walks (build_plan_pk): records of walk 0 are [0, pkb1),
    // of walk 1 [pkb1, P); first row word of each walk
    int pkb1, pkw0[2];
    const int *dtab;  // deep rows' per-column counts (cur[] after the plan, deep_table)
    unsigned long long key, gkey;
    int red[2 * NWARP + 2];
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

// The same unranking from shared tables T2[y] = C(y,2), T3[z] = C(z,3) (u32, exact), with a
// log2/exp2 estimate: no 64-bit arithmetic on the hot path. The correction loops make it exact.
template <int K>
__device__ __forceinline__ void unrank_tab(uint32_t r, int n, uint32_t M, const uint32_t *__restrict__ T2,
                                           const uint32_t *__restrict__ T3, int &a, int &b, int &c)
{
    if (K == 1) { a = (int)r; b = -1; c = -1; return; }
    uint32_t R = M - 1u - r;
    int top = n - 1;
    if (K == 3) {
        int z = (int)exp2f(__log2f(6.0f * (float)R + 1.0f) * (1.0f / 3.0f)) + 1;
        z = min(max(z, 2), top);
        while (T3[z] > R) z--;
        while (z < top && T3[z + 1] <= R) z++;
        R -= T3[z];
        a = n - 1 - z;
        top = z - 1;
    }
    int y = (int)((1.0f + sqrtf(8.0f * (float)R + 1.0f)) * 0.5f);
    y = min(max(y, 1), top);
    while (T2[y] > R) y--;
    while (y < top && T2[y + 1] <= R) y++;
    R -= T2[y];
    if (K == 2) { a = n - 1 - y; b = n - 1 - (int)R; c = -1; }
    else { b = n - 1 - y; c = n - 1 - (int)R; }
}

// Lexicographic successor of a sorted flip set (the last index varies fastest). Undefined past
// the last rank (never used there).
template <int K>
__device__ __forceinline__ void succ_flip(int n, int &a, int &b, int &c)
{
    if (K == 1) {
        ++a;
    } else if (K == 2) {
        if (++b == n) { ++a; b = a + 1; }
    } else {
        if (++c == n) {
            if (++b == n - 1) { ++a; b = a + 1; }
            c = b + 1;
        }
    }
}

// The low word of a selection key: the rank r, or (enc_keys) the flip set itself packed so that
// its order is the lexicographic order of (a, b, c), i.e. the rank order (reading R6): a << 20 |
// b << 10 | c for k = 3 (n <= 1024), a << 16 | b for k = 2 (n <= 65536). The u64 MIN of
// (f << 32 | low) then picks the same neighbour, and the winner's flip set needs no unranking.
template <int K>
__device__ __forceinline__ uint32_t enc_flip(int a, int b, int c)
{
    if (K == 3) return ((uint32_t)a << 20) | ((uint32_t)b << 10) | (uint32_t)c;
    if (K == 2) return ((uint32_t)a << 16) | (uint32_t)b;
    return (uint32_t)a;
}

template <int K>
__device__ __forceinline__ void dec_flip(uint32_t e, int &a, int &b, int &c)
{
    if (K == 3) { a = (int)(e >> 20); b = (int)((e >> 10) & 1023u); c = (int)(e & 1023u); }
    else if (K == 2) { a = (int)(e >> 16); b = (int)(e & 0xffffu); c = -1; }
    else { a = (int)e; b = -1; c = -1; }
}

// lex_rank(a < b < c) = M - 1 - [C(n-1-a, 3) + C(n-1-b, 2) + (n-1-c)] from the shared tables
template <int K>
__device__ __forceinline__ uint32_t rank_tab(int n, uint32_t M, const uint32_t *T2, const uint32_t *T3, int a, int b,
                                             int c)
{
    if (K == 3) return M - 1u - (T3[n - 1 - a] + T2[n - 1 - b] + (uint32_t)(n - 1 - c));
    if (K == 2) return M - 1u - (T2[n - 1 - a] + (uint32_t)(n - 1 - b));
    return (uint32_t)a;
}

__device__ __forceinline__ void fill_tables(uint32_t *T2, uint32_t *T3, int n)
{
    for (int i = threadIdx.x; i < n; i += blockDim.x) {
        const uint64_t z = (uint64_t)i;
        T2[i] = (uint32_t)(z * (z - 1) / 2);
        T3[i] = i >= 2 ? (uint32_t)(z * (z - 1) * (z - 2) / 6) : 0u;
    }
}

__device__ __forceinline__ int warp_min_i(int v) {
    for (int o = 16; o; o >>= 1) v = min(v, __shfl_xor_sync(FULL, v, o));
    return v;
}
__device__ __forceinline__ int warp_max_i(int v) {
    for (int o = 16; o; o >>= 1) v = max(v, __shfl_xor_sync(FULL, v, o));
    return v;
}
// u64 warp minimum with two 32-bit warp reductions (REDUX): the least high word, then the least
// low word among the lanes holding it -- the same as the 64-bit minimum of (hi << 32 | lo)
__device__ __forceinline__ unsigned long long warp_min_k(unsigned long long v) {
    const uint32_t hi = (uint32_t)(v >> 32), lo = (uint32_t)v;
    const uint32_t mh = __reduce_min_sync(FULL, hi);
    const uint32_t ml = __reduce_min_sync(FULL, hi == mh ? lo : 0xffffffffu);
    return ((unsigned long long)mh << 32) | ml;
}

// Wait (one thread) until the monotonic counter *ctr reaches target (acquire, gpu scope). A
// persistent grid is co-resident by construction (cooperative launch), so this always ends; a
// plain launch (LNS_PLAIN_LAUNCH) on a busy device has no such guarantee, so the wait gives up
// after timeout_ns of %globaltimer and returns false (the run then fails with LNS_EPEER instead
// of hanging).
__device__ __forceinline__ bool spin_until_ge(const unsigned long long *ctr, unsigned long long target,
                                              long long timeout_ns)
{
    unsigned long long seen, t_start, t_now;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(seen) : "l"(ctr) : "memory");
    if (seen >= target) return true;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_start));
    for (;;) {
        asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(seen) : "l"(ctr) : "memory");
        if (seen >= target) return true;
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_now));
        if ((long long)(t_now - t_start) > timeout_ns) return false;
    }
}

// Value range of Y: every thread passes its partial (min, max); a __syncthreads, then warp 0 sets
// the lattice ps.vlo / Uc of the next plan; callers must __syncthreads before reading them. (Written with min and max,
// not min(-y): nvcc 12.9 miscompiled an unrolled "mx = min(mx, -y)" into a 3-input min that
// dropped one negation.)
template <int K>
__device__ __forceinline__ void range_publish(int mn, int mx, PlanScalars &ps)
{
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    mn = warp_min_i(mn); mx = warp_max_i(mx);
    if (lane == 0) { ps.red[warp] = mn; ps.red[NWARP + warp] = mx; }
    __syncthreads();
    if (warp == 0) {
        int a = lane < NWARP ? ps.red[lane] : INT_MAX, b = lane < NWARP ? ps.red[NWARP + lane] : INT_MIN;
        a = warp_min_i(a); b = warp_max_i(b);
        if (lane == 0) {
            ps.vlo = a;
            ps.Uc = (b - a) / 2 + 1;
        }
    }
}

// Plan step D: X[w][c], per (row word, column word) pair, lane l loads sorted row 32w+l's sign
// bits of columns 32cw..32cw+31 (rowAt[p] = -1 marks a hole) and a 5-round shuffle transpose turns
// rows into columns; zero cnt[] for the next plan.
// The transpose of warps w0, w0 + 1, .., w0 + nw - 1 (no barrier).
__device__ __forceinline__ void plan_transpose_warps(const DevInst &I, const uint32_t *Ar, unsigned char *sm,
                                                     const Smem &L, const PlanScalars &ps, uint32_t *X, int w0, int nw)
{
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int m = I.m, n = I.n, NWn = I.NWn;
    const uint32_t *vbs = (const uint32_t *)(sm + L.vb);
    const int *rowAt = (const int *)(sm + L.rowAt);
    const int Wp = ps.Wp;
    for (int pr = warp - w0; pr < Wp * NWn; pr += nw) {
        const int w = pr / NWn, cw = pr - w * NWn;
        const int p = 32 * w + lane;
        const int j = I.pad ? rowAt[p] : (p < m ? rowAt[p] : -1);
        uint32_t x = j >= 0 ? (Ar[(size_t)j * NWn + cw] ^ vbs[cw]) : 0u;
#pragma unroll
        for (int j = 16; j >= 1; j >>= 1) {
            const uint32_t mk = j == 16 ? 0x0000FFFFu : j == 8 ? 0x00FF00FFu : j == 4 ? 0x0F0F0F0Fu
                              : j == 2 ? 0x33333333u : 0x55555555u;
            const uint32_t y = __shfl_xor_sync(FULL, x, j);
            x = (lane & j) ? ((x & ~mk) | ((y & ~mk) >> j)) : ((x & mk) | ((y & mk) << j));
        }
        const int c = 32 * cw + lane;
        if (c < n) X[w * n + c] = x;
    }
}

__device__ __forceinline__ void plan_transpose(const DevInst &I, const uint32_t *Ar, unsigned char *sm, const Smem &L,
                                               const PlanScalars &ps, uint32_t *X, int Uc)
{
    int *cnt = (int *)(sm + L.cnt);
    for (int u = threadIdx.x; u < Uc; u += NT) cnt[u] = 0;
    plan_transpose_warps(I, Ar, sm, L, ps, X, 0, NWARP);
    __syncthreads();
    PH(3);
}

// A pending move (the previous iteration's accepted flip set), applied by the next plan's step A
// while it counts the rows: Y'_j = Y_j - 2 sum_{i in F} B_ji, B_ji = V_i A_ji;
// thread 0 flips V's bits after step A's barrier (step D is the next reader of V).
struct Move {
    int on, a, b, c;
};

template <int K>
__device__ __forceinline__ int move_delta(const uint32_t *__restrict__ ar, const uint32_t *__restrict__ vbs, const Move &mv)
{
    int d = (((ar[mv.a >> 5] ^ vbs[mv.a >> 5]) >> (mv.a & 31)) & 1u) ? -1 : 1;
    if (K >= 2) d += (((ar[mv.b >> 5] ^ vbs[mv.b >> 5]) >> (mv.b & 31)) & 1u) ? -1 : 1;
    if (K == 3) d += (((ar[mv.c >> 5] ^ vbs[mv.c >> 5]) >> (mv.c & 31)) & 1u) ? -1 : 1;
    return d;
}

// Step A of both plan builders: apply the pending move to Y and count the rows per lattice point.
template <int K>
__device__ __forceinline__ void plan_count(const DevInst &I, const uint32_t *Ar, int *Ys, const uint32_t *vbs,
                                           int *cnt, int vlo, const Move &mv)
{
    for (int j = threadIdx.x; j < I.m; j += NT) {
        int y = Ys[j];
        if (mv.on) {
            y -= 2 * move_delta<K>(Ar + (size_t)j * I.NWn, vbs, mv);
            Ys[j] = y;
        }
        atomicAdd(&cnt[(y - vlo) >> 1], 1);
    }
}

__device__ __forceinline__ void flip_bits(uint32_t *vbs, int K, const Move &mv)
{
    vbs[mv.a >> 5] ^= 1u << (mv.a & 31);
    if (K >= 2) vbs[mv.b >> 5] ^= 1u << (mv.b & 31);
    if (K == 3) vbs[mv.c >> 5] ^= 1u << (mv.c & 31);
}

// ------------------------------------------------------------------------------------------
// Plan of the packed path (m <= 255, every bin count fits a byte), DESIGN.md §5.9. A row at lattice
// point u moves to bin u + 2t (t = #{i in F : x_ji = 1}), so bins of one parity of u only receive
// rows of that parity: the walked points [uneg, utop) split into two independent WALKS, walk p =
// points uneg + p, uneg + p + 2, ... In half-lattice units a point's rows land in its own bin and
// the next K bins of its walk, so a walk's open bins fit the four bytes of ONE 32-bit window.
// Row order: deep points (u < uneg, all destinations negative: linear cost, no records), walk 0,
// walk 1 (segments padded so that one of <= 32 rows never straddles a row word when I.pad), then
// the points above the top cut (no records; every such row costs 1). Records (uint4), one per
// (point, row word) piece, in walk order:
//   final piece of point u: (mask, L(u + 8), H_b << 8 | 8, 0x4404 | w_b << 16), b = vmin + 2(u - K)
//   earlier pieces:         (mask, 0,        0,            0x4444)
// L(u + 8) = rows of the point four steps ahead in the same walk (0 past utop): the funnel shift that
// completes bin u inserts it as the window's new top byte. w_b = 60|b| - 1 for b < 0, else 0.
// pstart[w] = first record in row word w (INT_MAX if none).
// ------------------------------------------------------------------------------------------
template <int K, bool XG = false, bool OVL = true>
__device__ void build_plan_pk(const DevInst &I, const uint32_t *Ar, unsigned char *sm, const Smem &L, PlanScalars &ps,
                              uint32_t *Xarg, const Move &mv, bool a_done = false)
{
    uint32_t *X = XG ? Xarg : (uint32_t *)(sm + L.X);
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int m = I.m, n = I.n;
    const int *Ys = (const int *)(sm + L.Y);
    const int *Hs = (const int *)(sm + L.H);
    int *cnt = (int *)(sm + L.cnt);
    int *seg = (int *)(sm + L.seg);
    int *cur = (int *)(sm + L.cur);
    int *pofs = (int *)(sm + L.pofs);
    int *rowAt = (int *)(sm + L.rowAt);
    int2 *bins = (int2 *)(sm + L.bins);
    uint4 *pk = (uint4 *)(sm + L.pk);
    int *pstart = (int *)(sm + L.pstart);
    const int vlo = ps.vlo, Uc = ps.Uc;

    // A. pending move; counting sort over the conservative lattice; holes; no record starts yet
    //    (a_done: the caller ran the counting sort and its barrier, build_plan for m > 255)
    if (!a_done) {
        plan_count<K>(I, Ar, (int *)Ys, (const uint32_t *)(sm + L.vb), cnt, vlo, mv);
        if (I.pad) for (int p = tid; p < 32 * I.XW; p += NT) rowAt[p] = -1;
    }
    for (int w = tid; w <= I.XW; w += NT) pstart[w] = -1;  // = 0xffffffff: no record (addresses, unsigned)
    __syncthreads();  // also: every thread has read ps.vlo / Uc before step B rewrites them
    PH(0);
    // B. warp 0: exact range, cuts, and the placement in the order deep | walk 0 | walk 1 | top
    if (tid == 0 && mv.on) flip_bits((uint32_t *)(sm + L.vb), K, mv);
    if (warp == 0) {
        int uf = -1, ul = -1;
        for (int b0 = 0; b0 < Uc; b0 += 32) {
            const unsigned bal = __ballot_sync(FULL, b0 + lane < Uc && cnt[b0 + lane] > 0);
            if (bal) {
                if (uf < 0) uf = b0 + __ffs(bal) - 1;
                ul = b0 + 31 - __clz(bal);
            }
        }
        const int U = ul - uf + 1;
        const int vmin = vlo + 2 * uf;
        int uneg = (-2 * K - vmin + 1) >> 1;  // least u with vmin + 2u >= -2K
        uneg = min(max(uneg, 0), U);
        int utop = ((I.maxS + 2 * K - vmin) >> 1) + 1;  // least u with vmin + 2u > maxS + 2K
        utop = min(max(utop, uneg), U);
        const int n0 = (utop - uneg + 1) >> 1;  // points of walk 0 (walk 1: the rest of [uneg, utop))
        // the placement is sequential (padding depends on the position within the row word), so
        // one thread walks the points: deep (contiguous), walk 0, walk 1 (padded), top (contiguous)
        int pos = 0, runp = 0, rneg = 0, rtop = 0, pkb1 = 0;
        if (!I.pad) {
            // unpadded: positions and record offsets are prefix sums (warp scans over the points in
            // placement order); an empty point is absorbed only by a non-empty predecessor here
            int sel = 0;  // lane holding q == uneg / uneg + n0 / utop: bits 0 / 1 / 2
            for (int q0 = 0; q0 < U; q0 += 32) {
                const int q = q0 + lane;
                const bool valid = q < U;
                const int v = q < uneg ? q : q < uneg + n0 ? uneg + 2 * (q - uneg)
                            : q < utop ? uneg + 1 + 2 * (q - uneg - n0) : q;
                const int Lq = valid ? cnt[uf + v] : 0;
                const bool walk = valid && q >= uneg && q < utop;
                const bool absorbed = walk && Lq == 0 && v - 2 >= uneg && vmin + 2 * (v - 2 - K) >= 0 &&
                                      cnt[uf + v - 2] > 0;
                int inc = Lq;
                for (int o = 1; o < 32; o <<= 1) { const int t_ = __shfl_up_sync(FULL, inc, o); if (lane >= o) inc += t_; }
                const int st = pos + inc - Lq, en = st + Lq;
                const int np = walk ? (Lq > 0 ? ((en - 1) >> 5) - (st >> 5) + 1 : (absorbed ? 0 : 1)) : 0;
                int incp = np;
                for (int o = 1; o < 32; o <<= 1) { const int t_ = __shfl_up_sync(FULL, incp, o); if (lane >= o) incp += t_; }
                const int p0 = runp + incp - np;
                if (valid) { seg[v] = st; cur[uf + v] = st; pofs[v] = absorbed ? -1 : p0; }
                if (q == uneg) { rneg = st; sel |= 1; }
                if (q == uneg + n0) { pkb1 = p0; sel |= 2; }
                if (q == utop) { rtop = st; sel |= 4; }
                pos += __shfl_sync(FULL, inc, 31);
                runp += __shfl_sync(FULL, incp, 31);
            }
            PH(7);
            // broadcast to lane 0 (the cuts at q = U take the totals)
            const unsigned b1 = __ballot_sync(FULL, sel & 1), b2 = __ballot_sync(FULL, sel & 2), b4 = __ballot_sync(FULL, sel & 4);
            rneg = b1 ? __shfl_sync(FULL, rneg, __ffs(b1) - 1) : pos;
            pkb1 = b2 ? __shfl_sync(FULL, pkb1, __ffs(b2) - 1) : runp;
            rtop = b4 ? __shfl_sync(FULL, rtop, __ffs(b4) - 1) : pos;
        } else if (lane == 0) {
            for (int v = 0; v < uneg; v++) {
                const int Lv = cnt[uf + v];
                seg[v] = pos; cur[uf + v] = pos; pofs[v] = 0;
                pos += Lv;
            }
            rneg = pos;
            int rows = pos;
            for (int q = 0; q < 2; q++) {
                if (q == 1) pkb1 = runp;
                int prev = 0;  // 2: the previous point's record may absorb this one
#pragma unroll 4
                for (int v = uneg + q; v < utop; v += 2) {
                    const int Lv = cnt[uf + v];
                    // m > 255: X may have fewer than 2W + 1 words, so a pad is taken only while the
                    // rows still to place fit (m <= 255: X has 2W + 1 words, every pad fits)
                    if (I.pad && Lv > 0 && (pos & 31) != 0 && (pos & 31) + Lv > 32 &&
                        (m <= PACKED_MAX_M || ((((pos + 31) & ~31) + (m - rows) + 31) >> 5) <= I.XW))
                        pos = (pos + 31) & ~31;
                    // an empty point whose bin and its predecessor's are non-negative is absorbed:
                    // the predecessor's final record completes both bins (no record of its own)
                    const bool nonneg = vmin + 2 * (v - K) >= 0;
                    const bool absorbed = Lv == 0 && nonneg && prev == 2;
                    seg[v] = pos; cur[uf + v] = pos; pofs[v] = absorbed ? -1 : runp;
                    runp += Lv > 0 ? ((pos + Lv - 1) >> 5) - (pos >> 5) + 1 : (absorbed ? 0 : 1);
                    prev = absorbed ? 1 : (nonneg ? 2 : 1);
                    pos += Lv;
                    rows += Lv;
                }
            }
            rtop = rows;
            for (int v = utop; v < U; v++) {
                const int Lv = cnt[uf + v];
                seg[v] = pos; cur[uf + v] = pos; pofs[v] = 0;
                pos += Lv;
            }
        }
        if (lane < 2) ps.pkw0[lane] = 0;  // (the walks' window constants: step C, warp 1)
        if (lane == 0) {
            ps.P = runp; ps.pkb1 = pkb1; ps.Wp = (pos + 31) >> 5;
            ps.vmin = vmin; ps.U = U; ps.NB = U + 2 * K; ps.ufirst = uf;
            ps.uneg = uneg; ps.utop = utop; ps.rneg = rneg; ps.rtop = rtop; ps.cneg = 0; ps.hwalk = 0;
            if (!a_done) ps.pkok = 1;
            ps.vlo = vmin - 2 * K; ps.Uc = U + 2 * K;
            ps.key = (unsigned long long)KEY_NONE;
            ps.gkey = (unsigned long long)KEY_NONE;
        }
    }
    __syncthreads();
    PH(1);
    // C. place rows; emit the records (one thread per walked point); bin constants; deep constant.
    //    pstart[w] = shared address of the first record in row word w
    const int vmin = ps.vmin, NB = ps.NB, uf = ps.ufirst, uneg = ps.uneg, utop = ps.utop;
    const uint32_t pk0 = (uint32_t)__cvta_generic_to_shared(pk);
    // OVL (one search, latency-bound): warps 2.. place the rows, meet at a named barrier and
    // transpose X (step D) while warp 0 builds the records and warp 1 the bin constants (neither
    // needs the placement). Batched searches place the rows first with every thread.
    if (!OVL) {
        for (int j = tid; j < m; j += NT) {
            const int p = atomicAdd(&cur[(Ys[j] - vlo) >> 1], 1);
            rowAt[p] = j;
        }
        __syncthreads();
    }
    PH(2);
    if (warp >= 2) {
        if (OVL) {
            for (int j = tid - 64; j < m; j += NT - 64) {
                const int p = atomicAdd(&cur[(Ys[j] - vlo) >> 1], 1);
                rowAt[p] = j;
            }
            asm volatile("bar.sync 1, %0;" ::"r"(NT - 64) : "memory");
        }
        plan_transpose_warps(I, Ar, sm, L, ps, X, 2, NWARP - 2);
    } else if (warp == 1) {
        // deep rows: 60 |b| per row at t = 0, minus 240 t (abs form); bin constants; H of the walked
        // bins (sums by warp reductions, no shared atomics)
        // walk q = lane (q = 0, 1): last point z, initial window (rows of the first four points),
        // trailing bins (the K bins past z: H bytes, one of them negative?) -> pkwt[q]
        int zq = -1;
        if (lane < 2) {
            const int n0 = (utop - uneg + 1) >> 1, n1 = (utop - uneg) >> 1;
            const int np = lane ? n1 : n0, a = uneg + lane, z = a + 2 * (np - 1);
            uint32_t win = 0, htr = 0;
            int trl = 0;
            if (np > 0) {
#pragma unroll
                for (int i = 0; i < 4; i++)
                    if (a + 2 * i <= z) win |= (uint32_t)cnt[uf + a + 2 * i] << (8 * i);
#pragma unroll
                for (int i = 1; i <= K; i++) {
                    const int b = vmin + 2 * (z + 2 * i - K);
                    if (b >= 0 && b <= n) htr |= (uint32_t)Hs[b] << (8 * (i - 1));
                    if (b < 0) trl = 1;
                }
            }
            zq = np > 0 ? z : -1;
            ps.pkwt[lane] = make_uint4(win, htr, (uint32_t)trl, (uint32_t)zq);
        }
        unsigned dneg = 0;
        for (int v = lane; v < uneg; v += 32)
            dneg += (unsigned)cnt[uf + v] * (unsigned)(60 * (2 * K - (vmin + 2 * v)));
        const int z0 = __shfl_sync(FULL, zq, 0), z1 = __shfl_sync(FULL, zq, 1);
        int hw = 0;
        for (int beta = lane; beta < NB; beta += 32) {
            const int b = vmin + 2 * (beta - K);
            const int Hb = (b >= 0 && b <= n) ? Hs[b] : 0;
            bins[beta] = make_int2(Hb, b < 0 ? 60 * (-b) - 1 : 0);
            // walked bins: [first point, last point + 2K] of the walk of beta's parity
            const int zp = ((beta - uneg) & 1) ? z1 : z0;
            if (Hb && beta >= uneg && zp >= 0 && beta <= zp + 2 * K) hw += Hb;
        }
        dneg = __reduce_add_sync(FULL, dneg);
        hw = __reduce_add_sync(FULL, hw);
        if (lane == 0) { ps.cneg = (int)dneg; ps.hwalk = hw; }
    } else {
        for (int v = uneg + lane; v < utop; v += 32) {
            const int st = seg[v], Lv = cnt[uf + v], en = st + Lv;
            int p = pofs[v];
            if (p < 0) continue;  // absorbed by its predecessor
            const int b = vmin + 2 * (v - K);
            uint32_t Hfin = ((b >= 0 && b <= n) ? (uint32_t)Hs[b] << 8 : 0u) | 8u;
            uint32_t wfin = 0x4404u | ((b < 0 ? (uint32_t)(60 * (-b) - 1) : 0u) << 16);
            uint32_t src = v + 8 < utop ? (uint32_t)cnt[uf + v + 8] : 0u;
            if (v + 2 < utop && pofs[v + 2] < 0) {
                // two bins: v and the absorbed v + 2 (both weights 0): h_v -> byte 1, h_v+2 -> byte 2 of
                // hb, H in bytes 1, 2 of z, shift 16 (the SAD adds 16 = 8 per bin), and the rows of the
                // points v + 8, v + 10 enter as the new bytes 2, 3
                const int b2 = b + 4;
                Hfin = (b2 <= n ? (uint32_t)Hs[b2] << 16 : 0u) | (b <= n ? (uint32_t)Hs[b] << 8 : 0u) | 16u;
                wfin = 0x4104u;
                src |= (v + 10 < utop ? (uint32_t)cnt[uf + v + 10] : 0u) << 8;
            }
            if (Lv == 0) {  // empty point: one zero record (in the previous row word) that completes its bin
                const int w = max(0, (st - 1) >> 5);
                pk[p] = make_uint4(0u, src, Hfin, wfin);
                atomicMin((unsigned *)&pstart[w], pk0 + 16u * p);
                if (v - uneg < 2) ps.pkw0[v - uneg] = w;
                continue;
            }
            const int w0 = st >> 5, w1 = (en - 1) >> 5;
            if (v - uneg < 2) ps.pkw0[v - uneg] = w0;
            for (int w = w0; w <= w1; w++, p++) {
                const int lo = max(st, 32 * w) - 32 * w, hi = min(en, 32 * w + 32) - 32 * w;
                const uint32_t mask = (hi == 32 ? FULL : ((1u << hi) - 1u)) & (FULL << lo);
                pk[p] = w == w1 ? make_uint4(mask, src, Hfin, wfin) : make_uint4(mask, 0u, 0u, 0x4444u);
                atomicMin((unsigned *)&pstart[w], pk0 + 16u * p);
            }
        }
        __syncwarp();  // the writers of pkw0 are in this warp
        PH(9);
        if (lane < 2) {  // the walks' ready-to-use addresses and constants (read by pk_walk)
            const int q = tid, wd = ps.pkw0[q];
            const int pb = q ? ps.pkb1 : 0, pe = q ? ps.P : ps.pkb1;
            const uint32_t xb = XG ? (uint32_t)(wd * n) : (uint32_t)__cvta_generic_to_shared(X + wd * n);
            ps.pkwk[q] = make_uint4(xb, pk0 + 16u * pb, pk0 + 16u * pe,
                                    (uint32_t)__cvta_generic_to_shared(pstart + wd + 1));
        }
    }
    __syncthreads();  // X (warps 2..), records, bins, pkwk / pkwt are published
    for (int u = tid; u < Uc; u += NT) cnt[u] = 0;  // zero for the next plan (its first barrier orders it)
    PH(3);
}

// ------------------------------------------------------------------------------------------
// Plan: per-iteration shared-memory structures of the current state (Y, V). Requires cnt[] = 0
// and a lattice ps.vlo / Uc covering every Y (the exact range after load_state, or the previous
// plan's range widened by 2k after a move: |Y'_j - Y_j| <= 2k). The exact range is found here.
//   cnt/cur   rows per conservative lattice point (Y = vlo + 2u)
//   seg       start of segment u - ufirst in sorted-row order (exact lattice, Y = vmin + 2u)
//   pieces    (mask, fin | w << 1 | len << 16): the part of one segment inside row word w, in row
//             order; fin = 1 on a segment's last piece (its bin is then complete); an empty
//             lattice point is one zero piece (mask 0, fin 1, len 0)
//   pstart    first piece of each row word
//   bins      (H_b, w_b) of bin beta <-> b = vmin + 2(beta - K): w_b = 60|b| - 1 for b < 0
//   X[w][c]   sign bits x_jc = [A_jc V_c = -1] of sorted rows 32w..32w+31, column c
// Leaves cnt[] zeroed, ps.key / gkey = KEY_NONE and ps.vlo / Uc set for the next plan.
// ------------------------------------------------------------------------------------------
template <int K, bool XG = false>
__device__ void build_plan_seg(const DevInst &I, const uint32_t *Ar, unsigned char *sm, const Smem &L, PlanScalars &ps,
                               uint32_t *Xarg, const Move &mv, bool a_done)
{
    uint32_t *X = XG ? Xarg : (uint32_t *)(sm + L.X);
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const int m = I.m, n = I.n;
    const int *Ys = (const int *)(sm + L.Y);
    const int *Hs = (const int *)(sm + L.H);
    int *cnt = (int *)(sm + L.cnt);
    int *seg = (int *)(sm + L.seg);
    int *cur = (int *)(sm + L.cur);
    int *pofs = (int *)(sm + L.pofs);
    int *rowAt = (int *)(sm + L.rowAt);
    int2 *bins = (int2 *)(sm + L.bins);
    uint2 *pieces = (uint2 *)(sm + L.pieces);
    int *pstart = (int *)(sm + L.pstart);
    const int vlo = ps.vlo, Uc = ps.Uc;

    // A. pending move; counting sort over the conservative lattice; holes of a padded placement
    if (!a_done) {
        plan_count<K>(I, Ar, (int *)Ys, (const uint32_t *)(sm + L.vb), cnt, vlo, mv);
        if (I.pad) for (int p = tid; p < 32 * I.XW; p += NT) rowAt[p] = -1;
    }
    __syncthreads();  // also: every thread has read ps.vlo / Uc before step B rewrites them
    PH(0);
    if (tid == 0 && mv.on) flip_bits((uint32_t *)(sm + L.vb), K, mv);
    // B. warp 0: exact range (first / last non-empty point), exclusive scans of the row and piece
    //    offsets over it, and the lattice of the next plan
    if (warp == 0) {
        int uf = -1, ul = -1;
        for (int b0 = 0; b0 < Uc; b0 += 32) {
            const unsigned bal = __ballot_sync(FULL, b0 + lane < Uc && cnt[b0 + lane] > 0);
            if (bal) {
                if (uf < 0) uf = b0 + __ffs(bal) - 1;
                ul = b0 + 31 - __clz(bal);
            }
        }
        const int U = ul - uf + 1;
        int runr = 0, runp = 0;
        for (int b0 = 0; b0 < U; b0 += 32) {
            const int v_ = b0 + lane;
            const int u = uf + v_;
            const int v = v_ < U ? cnt[u] : 0;
            int inc = v;
            for (int o = 1; o < 32; o <<= 1) { int t = __shfl_up_sync(FULL, inc, o); if (lane >= o) inc += t; }
            const int st = runr + inc - v, en = runr + inc;
            const int np = v_ < U ? (v > 0 ? ((en - 1) >> 5) - (st >> 5) + 1 : 1) : 0;  // empty point: one zero piece
            int incp = np;
            for (int o = 1; o < 32; o <<= 1) { int t = __shfl_up_sync(FULL, incp, o); if (lane >= o) incp += t; }
            if (v_ < U) { seg[v_] = st; cur[u] = st; pofs[v_] = runp + incp - np; }
            runr += __shfl_sync(FULL, inc, 31);
            runp += __shfl_sync(FULL, incp, 31);
        }
        // deep-negative prefix: points with value v < -2K (v = vlo + 2(uf + u))
        const int vmin_ = vlo + 2 * uf;
        int uneg = (-2 * K - vmin_ + 1) >> 1;  // least u with vmin + 2u >= -2K
        uneg = min(max(uneg, 0), U);
        int utop = ((I.maxS + 2 * K - vmin_) >> 1) + 1;  // least u with vmin + 2u > maxS + 2K
        utop = min(max(utop, uneg), U);
        int Wp = (m + 31) >> 5;
        __syncwarp();
        if (I.pad && lane == 0) {
            // budgeted padded placement: a walked segment that would straddle a
            // row word while starting mid-word starts at the next word, when the rows still to
            // place fit in the XW words X has even if nothing else is padded (fewer pieces, so
            // fewer POPCs per neighbour); deep rows stay contiguous at the front
            int pos = 0, left = m;
            runp = 0;
            for (int v = 0; v < U; v++) {
                const int Lv = cnt[uf + v];
                if (v >= uneg && v < utop && Lv > 0 && (pos & 31) != 0 && (pos & 31) + Lv > 32) {
                    const int np_ = (pos + 31) & ~31;
                    if (((np_ + left + 31) >> 5) <= I.XW) pos = np_;
                }
                seg[v] = pos; cur[uf + v] = pos; pofs[v] = runp;
                runp += Lv > 0 ? ((pos + Lv - 1) >> 5) - (pos >> 5) + 1 : 1;
                pos += Lv;
                left -= Lv;
            }
            runr = pos;
            Wp = (pos + 31) >> 5;
        }
        if (lane == 0) {
            const int vmin = vmin_;
            seg[U] = runr; pofs[U] = runp; ps.P = runp; pstart[Wp] = runp; ps.Wp = Wp;
            ps.vmin = vmin; ps.U = U; ps.NB = U + 2 * K; ps.ufirst = uf;
            ps.uneg = uneg; ps.utop = utop; ps.cneg = 0;
            if (!a_done) ps.pkok = 0;  // (a_done: set by build_plan, read by every thread)
            ps.vlo = vmin - 2 * K; ps.Uc = U + 2 * K;
            ps.key = (unsigned long long)KEY_NONE;
            ps.gkey = (unsigned long long)KEY_NONE;
        }
    }
    __syncthreads();
    PH(1);
    // C. place rows; emit pieces (one thread per segment); bin constants
    const int vmin = ps.vmin, U = ps.U, NB = ps.NB, uf = ps.ufirst;
    if (tid == 0) ps.rneg = seg[ps.uneg];
    for (int j = tid; j < m; j += NT) {
        const int p = atomicAdd(&cur[(Ys[j] - vlo) >> 1], 1);
        rowAt[p] = j;
    }
    const int uneg = ps.uneg;
    for (int v = tid; v < U; v += NT) {
        const int st = seg[v], en = st + cnt[uf + v];
        int p = pofs[v];
        // deep-negative constant sum_rows 60(2K - Y_j) - 1 (unsigned: the constant may exceed
        // 2^31 on its own; the fitness it enters does not)
        if (v < uneg && en > st)
            atomicAdd((unsigned *)&ps.cneg, (unsigned)(en - st) * (unsigned)(60 * (2 * K - (vmin + 2 * v)) - 1));
        if (st == en) {  // empty lattice point: a zero piece (in the previous row word) that finalises its bin
            pieces[p] = make_uint2(0u, 1u | ((uint32_t)((st - 1) >> 5) << 1));
            continue;
        }
        const int w0 = st >> 5, w1 = (en - 1) >> 5;
        for (int w = w0; w <= w1; w++, p++) {
            const int lo = max(st, 32 * w) - 32 * w, hi = min(en, 32 * w + 32) - 32 * w;
            const uint32_t mask = (hi == 32 ? FULL : ((1u << hi) - 1u)) & (FULL << lo);
            pieces[p] = make_uint2(mask, (uint32_t)(w == w1 ? 1 : 0) | ((uint32_t)w << 1) | ((uint32_t)(en - st) << 16));
            if (w > w0 || (st & 31) == 0) pstart[w] = p;
        }
    }
    for (int beta = tid; beta < NB; beta += NT) {
        const int b = vmin + 2 * (beta - K);
        const int Hb = (b >= 0 && b <= n) ? Hs[b] : 0;
        bins[beta] = make_int2(Hb, b < 0 ? 60 * (-b) - 1 : 0);
    }
    __syncthreads();
    PH(2);
    plan_transpose(I, Ar, sm, L, ps, X, Uc);
}

// The plan of the current state. m <= 255: the packed plan (every bin count fits a byte). m > 255
// with I.pkw: the packed plan whenever this state's counts still fit bytes, i.e.
// every byte the walk window can hold -- a walked bin's own rows plus the rows K points below it in
// its walk -- is <= 255, and so is H_b of every walked bin; else the segment plan. Decided per
// iteration by warp 0 after the shared counting sort.
template <int K, bool XG = false, bool OVL = true>
__device__ void build_plan_body(const DevInst &I, const uint32_t *Ar, unsigned char *sm, const Smem &L, PlanScalars &ps,
                                uint32_t *Xarg, const Move &mv);

// Deep rows' column table: the deep rows' cost is cneg - 240 sum t with
// sum t = sum_{i in F} #{deep rows j : x_ji = 1}, a sum of per-column counts, so once the plan's X
// is built every column's count D[c] is tabulated (in cur[], free between plans) and a neighbour
// reads k entries instead of walking the deep row words. Only when the deep rows span at least
// DEEP_TAB_MIN_W row words (one more barrier per plan).
#ifndef DEEP_TAB_MIN_W
#define DEEP_TAB_MIN_W 2
#endif
__device__ __forceinline__ bool deep_tab_on(int rneg) { return ((rneg + 31) >> 5) >= DEEP_TAB_MIN_W; }

template <bool XG>
__device__ __forceinline__ void deep_table(const DevInst &I, unsigned char *sm, const Smem &L, PlanScalars &ps,
                                           uint32_t *Xarg)
{
    const int rneg = ps.rneg;
    if (!deep_tab_on(rneg)) return;
    const uint32_t *X = XG ? Xarg : (const uint32_t *)(sm + L.X);
    int *D = (int *)(sm + L.cur);
    if (threadIdx.x == 0) ps.dtab = D;
    const int nw = (rneg + 31) >> 5, n = I.n;
    for (int col = threadIdx.x; col < n; col += NT) {
        int cntc = 0;
        for (int w = 0; w < nw; w++) {
            const uint32_t mask = (w == nw - 1 && (rneg & 31)) ? ((1u << (rneg & 31)) - 1u) : FULL;
            cntc += __popc(X[w * n + col] & mask);
        }
        D[col] = cntc;
    }
    __syncthreads();
}

template <int K, bool XG = false, bool OVL = true>
__device__ void build_plan(const DevInst &I, const uint32_t *Ar, unsigned char *sm, const Smem &L, PlanScalars &ps,
                           uint32_t *Xarg, const Move &mv = Move{0, 0, 0, 0})
{
    build_plan_body<K, XG, OVL>(I, Ar, sm, L, ps, Xarg, mv);
    deep_table<XG>(I, sm, L, ps, Xarg);
}

template <int K, bool XG, bool OVL>
__device__ void build_plan_body(const DevInst &I, const uint32_t *Ar, unsigned char *sm, const Smem &L, PlanScalars &ps,
                                uint32_t *Xarg, const Move &mv)
{
    if (I.m <= PACKED_MAX_M) { build_plan_pk<K, XG, OVL>(I, Ar, sm, L, ps, Xarg, mv); return; }
    if (!I.pkw) { build_plan_seg<K, XG>(I, Ar, sm, L, ps, Xarg, mv, false); return; }
    const int tid = threadIdx.x, lane = tid & 31;
    int *cnt = (int *)(sm + L.cnt);
    const int *Hs = (const int *)(sm + L.H);
    const int vlo = ps.vlo, Uc = ps.Uc;
    plan_count<K>(I, Ar, (int *)(sm + L.Y), (const uint32_t *)(sm + L.vb), cnt, vlo, mv);
    if (I.pad) for (int p = tid; p < 32 * I.XW; p += NT) ((int *)(sm + L.rowAt))[p] = -1;
    __syncthreads();
    if (tid < 32) {
        int uf = -1, ul = -1;
        for (int b0 = 0; b0 < Uc; b0 += 32) {
            const unsigned bal = __ballot_sync(FULL, b0 + lane < Uc && cnt[b0 + lane] > 0);
            if (bal) {
                if (uf < 0) uf = b0 + __ffs(bal) - 1;
                ul = b0 + 31 - __clz(bal);
            }
        }
        const int U = ul - uf + 1, vmin = vlo + 2 * uf;
        int uneg = (-2 * K - vmin + 1) >> 1;
        uneg = min(max(uneg, 0), U);
        int utop = ((I.maxS + 2 * K - vmin) >> 1) + 1;
        utop = min(max(utop, uneg), U);
        bool bad = false;
        for (int v = uneg + lane; v < utop + 2 * K; v += 32) {  // bins of both walks
            int s4 = 0;
            for (int t = 0; t <= K; t++) {
                const int p = v - 2 * t;
                if (p >= uneg && p < utop) s4 += cnt[uf + p];
            }
            const int b = vmin + 2 * (v - K);
            bad |= s4 > 255 || (b >= 0 && b <= I.n && Hs[b] > 255);
        }
        const bool anybad = __any_sync(FULL, bad);
        if (lane == 0) ps.pkok = anybad ? 0 : 1;
    }
    __syncthreads();
    if (ps.pkok) build_plan_pk<K, XG, OVL>(I, Ar, sm, L, ps, Xarg, mv, true);
    else build_plan_seg<K, XG>(I, Ar, sm, L, ps, Xarg, mv, true);
}

// One lattice point (segment) of eval_fit: its pieces add POPC counts of the bit-sliced planes
// (reloading the lane's three column words only when the piece's row word changes); then its row
// counts N_t land in bins beta + 2t and bin beta is complete. Registers Ra.. hold bins
// beta .. beta+2K-1; the caller rotates the names (Ra becomes bin beta+2K), so no moves are needed.
template <int K>
__device__ __forceinline__ void seg_step(const uint2 *__restrict__ &pp, uint2 &rec, const int2 *__restrict__ &bp,
                                         const uint32_t *__restrict__ X, int n, int a, int b, int c, int &curw,
                                         uint32_t &lo, uint32_t &hi, uint32_t &lh, int &f, int &smin,
                                         int &Ra, int &Rc, int &Re)
{
    int c1 = 0, c2 = 0, c3 = 0;
    const int2 bn = *bp++;  // this segment's bin constants, loaded early
    uint2 cur;
    do {
        // rec holds the current piece (prefetched); fetch the next one before using it (the piece
        // list is padded, so reading one past the last piece is safe)
        cur = rec;
        rec = *++pp;
        const int w = (int)((cur.y >> 1) & 0x7fffu);
        if (w != curw) {
            curw = w;
            const uint32_t *xr = X + w * n;
            if (K == 1) {
                lo = xr[a];
            } else if (K == 2) {
                const uint32_t xa = xr[a], xb = xr[b];
                lo = xa ^ xb; hi = xa & xb;
            } else {
                const uint32_t xa = xr[a], xb = xr[b], xc = xr[c];
                lo = xa ^ xb ^ xc;
                hi = (xa & xb) | (xc & (xa ^ xb));
                lh = lo & hi;
            }
        }
        c1 += __popc(lo & cur.x);
        if (K >= 2) c2 += __popc(hi & cur.x);
        if (K == 3) c3 += __popc(lh & cur.x);
    } while (!(cur.y & 1u));
    const int len = (int)(cur.y >> 16);
    int h;
    if (K == 1) {         // N1 = c1 -> bin beta+2 (reuses Ra)
        h = Ra + len - c1;
        Ra = c1;
    } else if (K == 2) {  // N1 = c1 -> beta+2 (Rc), N2 = c2 -> beta+4 (Ra)
        h = Ra + len - c1 - c2;
        Rc += c1; Ra = c2;
    } else {              // N1 = c1-c3 -> beta+2 (Rc), N2 = c2-c3 -> beta+4 (Re), N3 = c3 -> beta+6 (Ra)
        h = Ra + len - c1 - c2 + c3;
        Rc += c1 - c3; Re += c2 - c3; Ra = c3;
    }
    f += bn.y * h;
    smin += min(h, bn.x);
}

__device__ __forceinline__ void bin_cost(int h, int2 bn, int &f, int &smin)
{
    f += bn.y * h;
    smin += min(h, bn.x);
}

// Fitness of neighbour (a, b, c) from the plan, segment-major over the U lattice points:
//   f = 2m + sum_beta ( w_beta h_beta - 2 min(h_beta, H_beta) )
// (|h - H| = h + H - 2 min(h, H) summed over b = 0..n; every row lands in exactly one bin.)
struct EvalRange {
    int u0, u1;       // lattice points [u0, u1) go through the segment loop (u0 = uneg, u1 = utop)
    int rneg, cneg;   // deep-negative rows [0, rneg) and their constant part
    int p0;           // first piece of point u0
    const int *dtab;  // deep rows' per-column counts (deep_table), used when deep_tab_on(rneg)
};

// Deep-negative rows: every destination is negative, cost sum_j 60(2K - Y_j - 4 t_j) - 1
//   = cneg - 240 sum_j t_j, with sum t = popc(lo) + 2 popc(hi) over their (sorted) row words.
template <int K>
__device__ __forceinline__ int deep_negative(const uint32_t *__restrict__ X, int n, const EvalRange &er, int f,
                                             int a, int b, int c)
{
    int st = 0;
    if (deep_tab_on(er.rneg)) {  // sum t = sum over the flipped columns of their deep-row counts
        st = er.dtab[a];
        if (K >= 2) st += er.dtab[b];
        if (K == 3) st += er.dtab[c];
        return (int)((unsigned)f + (unsigned)er.cneg - 240u * (unsigned)st);
    }
    const int nw = (er.rneg + 31) >> 5;
    for (int w = 0; w < nw; w++) {
        const uint32_t mask = (w == nw - 1 && (er.rneg & 31)) ? ((1u << (er.rneg & 31)) - 1u) : FULL;
        const uint32_t *xr = X + w * n;
        if (K == 1) {
            st += __popc(xr[a] & mask);
        } else if (K == 2) {
            const uint32_t xa = xr[a], xb = xr[b];
            st += __popc((xa ^ xb) & mask) + 2 * __popc(xa & xb & mask);
        } else {
            const uint32_t xa = xr[a], xb = xr[b], xc = xr[c];
            st += __popc((xa ^ xb ^ xc) & mask) + 2 * __popc(((xa & xb) | (xc & (xa ^ xb))) & mask);
        }
    }
    return (int)((unsigned)f + (unsigned)er.cneg - 240u * (unsigned)st);
}

template <int K, bool DEEP>
__device__ __forceinline__ int eval_fit(const uint32_t *__restrict__ X, const uint2 *__restrict__ pieces,
                                        const int2 *__restrict__ bins, int n, const EvalRange &er, int m2,
                                        int a, int b, int c)
{
    int f = m2, smin = 0;
    if (DEEP) f = deep_negative<K>(X, n, er, f, a, b, c);
    const int U = er.u1 - er.u0;
    if (U <= 0) return f;
    int R0 = 0, R1 = 0, R2 = 0, R3 = 0, R4 = 0, R5 = 0;
    int curw = -1;
    uint32_t lo = 0, hi = 0, lh = 0;
    const uint2 *pp = pieces + er.p0;
    uint2 rec = *pp;
    const int2 *bp = bins + er.u0;
    int u = 0;
#define SEG(Ra, Rc, Re) seg_step<K>(pp, rec, bp, X, n, a, b, c, curw, lo, hi, lh, f, smin, Ra, Rc, Re)
#define TRAIL2(A, B) { bin_cost(A, bp[0], f, smin); bin_cost(B, bp[1], f, smin); }
#define TRAIL4(A, B, C, D) { TRAIL2(A, B) bin_cost(C, bp[2], f, smin); bin_cost(D, bp[3], f, smin); }
#define TRAIL6(A, B, C, D, E, F) { TRAIL4(A, B, C, D) bin_cost(E, bp[4], f, smin); bin_cost(F, bp[5], f, smin); }
    if (K == 1) {
        for (;;) {
            SEG(R0, R0, R0); if (++u == U) { TRAIL2(R1, R0); break; }
            SEG(R1, R1, R1); if (++u == U) { TRAIL2(R0, R1); break; }
        }
    } else if (K == 2) {
        for (;;) {
            SEG(R0, R2, R0); if (++u == U) { TRAIL4(R1, R2, R3, R0); break; }
            SEG(R1, R3, R1); if (++u == U) { TRAIL4(R2, R3, R0, R1); break; }
            SEG(R2, R0, R2); if (++u == U) { TRAIL4(R3, R0, R1, R2); break; }
            SEG(R3, R1, R3); if (++u == U) { TRAIL4(R0, R1, R2, R3); break; }
        }
    } else {
        for (;;) {
            SEG(R0, R2, R4); if (++u == U) { TRAIL6(R1, R2, R3, R4, R5, R0); break; }
            SEG(R1, R3, R5); if (++u == U) { TRAIL6(R2, R3, R4, R5, R0, R1); break; }
            SEG(R2, R4, R0); if (++u == U) { TRAIL6(R3, R4, R5, R0, R1, R2); break; }
            SEG(R3, R5, R1); if (++u == U) { TRAIL6(R4, R5, R0, R1, R2, R3); break; }
            SEG(R4, R0, R2); if (++u == U) { TRAIL6(R5, R0, R1, R2, R3, R4); break; }
            SEG(R5, R1, R3); if (++u == U) { TRAIL6(R0, R1, R2, R3, R4, R5); break; }
        }
    }
#undef SEG
#undef TRAIL2
#undef TRAIL4
#undef TRAIL6
    return f - 2 * smin;
}

// ---- packed path (m <= 255), parity walks (build_plan_pk) ------------------
// A walk's open bins live in the four bytes of one 32-bit window w: byte i = bin u + 2i of the
// walk (u = the point being processed), initialised with the rows of those points ("len") and
// receiving each point's rows as they move: a piece with row counts c1 = |lo & mask|,
// c2 = |hi & mask|, c3 = |lh & mask| moves N1 = c1 - c3 rows to byte 1, N2 = c2 - c3 to byte 2 and
// N3 = c3 to byte 3, all out of byte 0:
//   w += 255 N1 + 65535 N2 + 16777215 N3 = 255 c1 + 65535 c2 + 16711425 c3      (K = 3)
// Bytes may go transiently negative inside the register; it is exact modulo 2^32 and every byte
// is a count in [0, 255] whenever it is read or shifted. The final piece of a point completes
// bin u (byte 0): f += w_b h + |h - H_b| (+ 8, taken out of the constant C), and the funnel shift
// by 8 drops it and inserts the rows of the point four steps ahead as the new top byte.
template <int K>
__device__ __forceinline__ void load_planes(const uint32_t *__restrict__ xr, int a, int b, int c, uint32_t &lo,
                                            uint32_t &hi, uint32_t &lh)
{
    if (K == 1) {
        lo = xr[a]; hi = 0; lh = 0;
    } else if (K == 2) {
        const uint32_t xa = xr[a], xb = xr[b];
        lo = xa ^ xb; hi = xa & xb; lh = 0;
    } else {
        const uint32_t xa = xr[a], xb = xr[b], xc = xr[c];
        lo = xa ^ xb ^ xc;
        hi = (xa & xb) | (xc & (xa ^ xb));
        lh = lo & hi;
    }
}

#ifndef PK_TWO_PLANES
#define PK_TWO_PLANES 1  // c3 = |lo & hi & mask| by one three-input LOP3 (no lh register per neighbour)
#endif
template <int K>
__device__ __forceinline__ void pk_step(const uint4 &r, uint32_t lo, uint32_t hi, uint32_t lh, uint32_t &w, int &f)
{
    // (c3 first: with this order ptxas's register assignment of the record loop avoids the dispatch
    // stalls the c1, c2, c3 order showed in the batched kernel)
    if (K == 3) w += 16711425u * (uint32_t)__popc((PK_TWO_PLANES ? lo & hi : lh) & r.x);
    if (K >= 2) w += 65535u * (uint32_t)__popc(hi & r.x);
    w += 255u * (uint32_t)__popc(lo & r.x);
    // hb: byte 1 = h (byte 0 of w) for a final piece (selector 0x4404), 0 otherwise (0x4444)
    uint32_t hb, fu = (uint32_t)f;
    asm("prmt.b32 %0, %1, %2, %3;" : "=r"(hb) : "r"(w), "r"(0u), "r"(r.w));
    fu = __dp2a_lo(r.w, hb, fu);  // + w_b h (w_b in the high half of r.w; the selector meets byte 0 = 0)
    asm("vabsdiff4.u32.u32.u32.add %0, %1, %2, %3;" : "=r"(fu) : "r"(hb), "r"(r.z), "r"(fu));  // + |h - H_b| + shift
    f = (int)fu;
    w = __funnelshift_r(w, r.y, r.z);  // shift r.z & 31 (8 or 0); r.y byte 0 enters as byte 3
}

// The packed plan's scalars are read from shared memory (PlanScalars) where they are used, which
// keeps them out of the registers of the record loop.
// The K bins past a walk's last point hold only carried rows (bytes 0 .. K-1 of w; the rest are
// 0): sum |h - H| is one SAD against the packed H, unless one of them is negative (w_b != 0).
template <int K>
__device__ __forceinline__ void pk_trail(const uint4 &wt, const int2 *__restrict__ bins, uint32_t w, int &f)
{
    if (!wt.z) {
        f += (int)__vsadu4(w, wt.y);
        return;
    }
#pragma unroll
    for (int i = 0; i < K; i++) {
        const int h = (int)((w >> (8 * i)) & 0xffu);
        const int2 bn = bins[(int)wt.w + 2 * (i + 1)];
        f += bn.y * h + abs(h - bn.x);
    }
}

// Column words of one row word: LDS from the 32-bit shared address xs (XG = false), or plain loads
// from the global-memory X of very large instances (XG = true, xg).
template <int K, bool XG>
__device__ __forceinline__ void pk_planes(const uint32_t *__restrict__ xg, uint32_t xs, int a, int b, int c,
                                          uint32_t &lo, uint32_t &hi, uint32_t &lh)
{
    uint32_t xa, xb = 0, xc = 0;
    if (XG) {
        xa = xg[a];
        if (K >= 2) xb = xg[b];
        if (K == 3) xc = xg[c];
    } else {
        asm("ld.shared.u32 %0, [%1];" : "=r"(xa) : "r"(xs + 4u * a));
        if (K >= 2) asm("ld.shared.u32 %0, [%1];" : "=r"(xb) : "r"(xs + 4u * b));
        if (K == 3) asm("ld.shared.u32 %0, [%1];" : "=r"(xc) : "r"(xs + 4u * c));
    }
    if (K == 1) {
        lo = xa; hi = 0; lh = 0;
    } else if (K == 2) {
        lo = xa ^ xb; hi = xa & xb; lh = 0;
    } else {
        lo = xa ^ xb ^ xc;
        hi = (xa & xb) | (xc & (xa ^ xb));
        lh = PK_TWO_PLANES ? 0u : lo & hi;
    }
}

// One walk q of NB neighbours (NB = 1 or 2, the second in a1, b1, c1): word-major (the lane's
// column words are loaded once per row word), the record stream shared by the neighbours. All
// addresses are 32-bit shared-window addresses prepared by build_plan_pk (the asm loads read plan
// memory that only changes across the plan's barriers, and every address derives from a fresh
// load of pkwk, so no load can be reused across plans).
template <int K, int NB, bool XG>
__device__ __forceinline__ void pk_walk(const PlanScalars &ps, int q, const uint32_t *__restrict__ X,
                                        const int2 *__restrict__ bins, int n, int a0, int b0, int c0, int a1, int b1,
                                        int c1, int &f0, int &f1)
{
    const uint4 wk = ps.pkwk[q];
    if (wk.y == wk.z) return;
    const uint4 wt = ps.pkwt[q];
    uint32_t w0 = wt.x, w1 = wt.x;
    uint32_t pp = wk.y, pw = wk.w, xs = wk.x;
    const uint32_t pe = wk.z;
    const uint32_t *xg = XG ? X + wk.x : nullptr;
    for (;;) {
        uint32_t lo0, hi0, lh0, lo1 = 0, hi1 = 0, lh1 = 0;
        pk_planes<K, XG>(xg, xs, a0, b0, c0, lo0, hi0, lh0);
        if (NB == 2) pk_planes<K, XG>(xg, xs, a1, b1, c1, lo1, hi1, lh1);
        if (XG) xg += n; else xs += 4u * n;
        uint32_t pend;
        asm("ld.shared.u32 %0, [%1];" : "=r"(pend) : "r"(pw));
        pw += 4u;
        pend = min(pend, pe);
#pragma unroll kPkUnroll
        for (; pp < pend; pp += 16u) {
            uint4 r;
            asm("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];" : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w) : "r"(pp));
            pk_step<K>(r, lo0, hi0, lh0, w0, f0);
            if (NB == 2) pk_step<K>(r, lo1, hi1, lh1, w1, f1);
        }
        if (pend == pe) break;
    }
    pk_trail<K>(wt, bins, w0, f0);
    if (NB == 2) pk_trail<K>(wt, bins, w1, f1);
}

// Deep rows (DEEP): every destination negative, cost cneg - 240 sum t (abs form).
template <int K>
__device__ __forceinline__ int pk_deep(const uint32_t *__restrict__ X, int n, const PlanScalars &ps, int f, int a,
                                       int b, int c)
{
    EvalRange er;
    er.rneg = ps.rneg; er.cneg = ps.cneg; er.dtab = ps.dtab;
    return deep_negative<K>(X, n, er, f, a, b, c);
}

template <int K, int NB, bool DEEP, bool XG>
__device__ __forceinline__ void eval_pk(const PlanScalars &ps, int cabs, const uint32_t *__restrict__ X,
                                        const uint4 *__restrict__ pk, const int *__restrict__ pstart,
                                        const int2 *__restrict__ bins, int n, int a0, int b0, int c0, int a1, int b1,
                                        int c1, int &f0, int &f1)
{
    f0 = cabs;
    if (NB == 2) f1 = cabs;
    if (DEEP) {
        f0 = pk_deep<K>(X, n, ps, f0, a0, b0, c0);
        if (NB == 2) f1 = pk_deep<K>(X, n, ps, f1, a1, b1, c1);
    }
    pk_walk<K, NB, XG>(ps, 0, X, bins, n, a0, b0, c0, a1, b1, c1, f0, f1);
    pk_walk<K, NB, XG>(ps, 1, X, bins, n, a0, b0, c0, a1, b1, c1, f0, f1);
}

// Evaluate ranks [blo, bhi) (blo 32-aligned) of this CTA at iteration t; returns this thread's best
// key. until (nullable) is indexed by r - ubase: rank r is tabu iff until[r - ubase] >= t.
template <int K, bool WRITE_ALL, bool XG = false>
__device__ unsigned long long eval_range(const DevInst &I, const unsigned char *sm, const Smem &L,
                                         const PlanScalars &ps, const uint32_t *Xarg, uint32_t M, uint32_t blo, uint32_t bhi,
                                         const uint32_t *until, uint32_t ubase, uint32_t t, int32_t *fit_out,
                                         const uint2 *tri = nullptr, int aspire = 0,
                                         int best_f = 0, const uint32_t *tbits = nullptr, bool enc = false)
{
    // rank r tabu at iteration t: the until[] array (smem slice or global), or the bitmap
    auto is_tabu = [&](uint32_t r) -> bool {
        if (until) return until[r - ubase] >= t;
        // plain (L1-coherent) load: the CTA's own thread 0 updates these words between iterations
        return tbits && ((tbits[r >> 5] >> (r & 31)) & 1u);
    };
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    // X from the shared window when it lives there, so the compiler emits LDS (not generic loads)
    const uint32_t *X = XG ? Xarg : (const uint32_t *)(sm + L.X);
    const uint2 *pieces = (const uint2 *)(sm + L.pieces);
    const int2 *bins = (const int2 *)(sm + L.bins);
    const uint32_t *T2 = (const uint32_t *)(sm + L.T2), *T3 = (const uint32_t *)(sm + L.T3);
    const bool packed = ps.pkok;
    EvalRange er;
    er.u0 = ps.uneg; er.u1 = ps.utop; er.rneg = ps.rneg; er.cneg = ps.cneg; er.dtab = (const int *)(sm + L.cur);
    er.p0 = ((const int *)(sm + L.pofs))[ps.uneg];
    // packed path, abs form: C = m - (H of the walked bins) + (rows above the top cut) - 8 (completed
    // bins); deep rows cost 60 |b| each (cneg, accumulated so by build_plan_pk)
    const int cabs = packed ? 2 * I.m - ps.hwalk - ps.rtop - 8 * (ps.utop - ps.uneg) : 0;
    const int *pstart = (const int *)(sm + L.pstart);
    const uint4 *pk = (const uint4 *)(sm + L.pk);
    unsigned long long best = (unsigned long long)KEY_NONE;
    if (packed && PK_PAIR && !tri && bhi - blo >= 4u * NT) {
        // large slices (batched searches): each thread owns a contiguous run of ranks, split into
        // halves A and B evaluated as a pair; flip sets advance by lexicographic successor, so
        // only the two run starts are unranked
        const uint32_t span = bhi - blo, tid = threadIdx.x;
        const uint32_t lo = blo + (uint32_t)(((uint64_t)span * tid) / NT);
        const uint32_t hi = blo + (uint32_t)(((uint64_t)span * (tid + 1)) / NT);
        const uint32_t mid = lo + (hi - lo + 1) / 2;
        int a0, b0, c0, a1, b1, c1;
        unrank_tab<K>(lo, I.n, M, T2, T3, a0, b0, c0);
        if (mid < hi) unrank_tab<K>(mid, I.n, M, T2, T3, a1, b1, c1);
        else { a1 = a0; b1 = b0; c1 = c0; }
        for (uint32_t rA = lo, rB = mid; rA < mid; ++rA, ++rB) {
            const bool vB = rB < hi;
            const uint32_t rb = vB ? rB : rA;
            if (!vB) { a1 = a0; b1 = b0; c1 = c0; }
            int fA, fB;
            if (ps.rneg > 0) eval_pk<K, 2, true, XG>(ps, cabs, X, pk, pstart, bins, I.n, a0, b0, c0, a1, b1, c1, fA, fB);
            else eval_pk<K, 2, false, XG>(ps, cabs, X, pk, pstart, bins, I.n, a0, b0, c0, a1, b1, c1, fA, fB);
            const bool tA = is_tabu(rA);
            const bool tB = is_tabu(rb);
            if (WRITE_ALL) { fit_out[rA] = fA; if (vB) fit_out[rB] = fB; }
            // (rank keys only: launch_search sets enc_keys only when no CTA takes this path)
            const unsigned long long kA = ((unsigned long long)(uint32_t)fA << 32) | rA;
            const unsigned long long kB = ((unsigned long long)(uint32_t)fB << 32) | rb;
            if ((!tA || (aspire && fA < best_f)) && kA < best) best = kA;
            if ((!tB || (aspire && fB < best_f)) && kB < best) best = kB;
            succ_flip<K>(I.n, a0, b0, c0);
            succ_flip<K>(I.n, a1, b1, c1);
        }
        return best;
    }
    if (packed && PK_PAIR && bhi - blo > (uint32_t)NT) {
        // two neighbours per thread: ranks r and r + 32 (a warp covers 64 consecutive ranks); only
        // when the slice needs more than one pass of the block, else half the warps would idle
        for (uint32_t r0 = blo + 64u * warp; r0 < bhi; r0 += 2 * NT) {
            const uint32_t rA = r0 + lane, rB = rA + 32u;
            if (rA >= bhi) continue;
            const bool vB = rB < bhi;
            const uint32_t rb = vB ? rB : rA;  // a ragged tail re-evaluates rA in the B slot
            int a0, b0, c0, a1, b1, c1;
            if (tri) {
                const uint2 q0 = tri[rA - blo], q1 = tri[rb - blo];
                a0 = (int)(q0.x & 0xffffu); b0 = (int)(q0.x >> 16); c0 = (int)q0.y;
                a1 = (int)(q1.x & 0xffffu); b1 = (int)(q1.x >> 16); c1 = (int)q1.y;
            } else {
                unrank_tab<K>(rA, I.n, M, T2, T3, a0, b0, c0);
                unrank_tab<K>(rb, I.n, M, T2, T3, a1, b1, c1);
            }
            int fA, fB;
            if (ps.rneg > 0) eval_pk<K, 2, true, XG>(ps, cabs, X, pk, pstart, bins, I.n, a0, b0, c0, a1, b1, c1, fA, fB);
            else eval_pk<K, 2, false, XG>(ps, cabs, X, pk, pstart, bins, I.n, a0, b0, c0, a1, b1, c1, fA, fB);
            const bool tA = is_tabu(rA);
            const bool tB = is_tabu(rb);
            if (WRITE_ALL) { fit_out[rA] = fA; if (vB) fit_out[rB] = fB; }
            const unsigned long long kA = ((unsigned long long)(uint32_t)fA << 32) | (enc ? enc_flip<K>(a0, b0, c0) : rA);
            const unsigned long long kB = ((unsigned long long)(uint32_t)fB << 32) | (enc ? enc_flip<K>(a1, b1, c1) : rb);
            if ((!tA || (aspire && fA < best_f)) && kA < best) best = kA;
            if ((!tB || (aspire && fB < best_f)) && kB < best) best = kB;
        }
        return best;
    }
    for (uint32_t r0 = blo + 32u * warp; r0 < bhi; r0 += NT) {
        const uint32_t r = r0 + lane;
        if (r < bhi) {
            const bool tab = is_tabu(r);
            if (!tab || WRITE_ALL || aspire) {
                int a, b, c;
                if (tri) {  // flip sets of this CTA's fixed slice, precomputed at launch
                    const uint2 q = tri[r - blo];
                    a = (int)(q.x & 0xffffu); b = (int)(q.x >> 16); c = (int)q.y;
                } else {
                    unrank_tab<K>(r, I.n, M, T2, T3, a, b, c);
                }
                int f, g_;
                if (packed) {
                    if (ps.rneg > 0) eval_pk<K, 1, true, XG>(ps, cabs, X, pk, pstart, bins, I.n, a, b, c, a, b, c, f, g_);
                    else eval_pk<K, 1, false, XG>(ps, cabs, X, pk, pstart, bins, I.n, a, b, c, a, b, c, f, g_);
                } else {
                    f = er.rneg > 0 ? eval_fit<K, true>(X, pieces, bins, I.n, er, 2 * I.m, a, b, c)
                                    : eval_fit<K, false>(X, pieces, bins, I.n, er, 2 * I.m, a, b, c);
                }
                if (WRITE_ALL) fit_out[r] = f;
                const unsigned long long key = ((unsigned long long)(uint32_t)f << 32) | (enc ? enc_flip<K>(a, b, c) : r);
                // admissible: not tabu, or (aspiration) better than the best fitness so far
                if ((!tab || (aspire && f < best_f)) && key < best) best = key;
            }
        }
    }
    return best;
}

// Apply the move F to the CTA's shared copy of (Y, V): Y'_j = Y_j - 2 sum_{i in F} B_ji,
// B_ji = V_i A_ji, then flip the bits of V. The flip is ordered before the
// next reads of V (plan step D) by the plan's own barriers.
template <int K>
__device__ void apply_move(const DevInst &I, const uint32_t *Ar, int *Ys, uint32_t *vbs, int a, int b, int c)
{
    for (int j = threadIdx.x; j < I.m; j += NT) {
        const uint32_t *ar = Ar + (size_t)j * I.NWn;
        int d = (((ar[a >> 5] ^ vbs[a >> 5]) >> (a & 31)) & 1u) ? -1 : 1;
        if (K >= 2) d += (((ar[b >> 5] ^ vbs[b >> 5]) >> (b & 31)) & 1u) ? -1 : 1;
        if (K == 3) d += (((ar[c >> 5] ^ vbs[c >> 5]) >> (c & 31)) & 1u) ? -1 : 1;
        Ys[j] -= 2 * d;
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        vbs[a >> 5] ^= 1u << (a & 31);
        if (K >= 2) vbs[b >> 5] ^= 1u << (b & 31);
        if (K == 3) vbs[c >> 5] ^= 1u << (c & 31);
    }
}

// Slice [blo, bhi) of CTA `b` of `nb` inside [lo, hi), boundaries on multiples of 32.
__device__ __forceinline__ void cta_slice(uint32_t lo, uint32_t hi, unsigned b, unsigned nb, uint32_t &blo, uint32_t &bhi)
{
    uint64_t span = hi - lo;
    blo = lo + 32u * (uint32_t)((span * b / nb) / 32);
    bhi = (b + 1 == nb) ? hi : lo + 32u * (uint32_t)((span * (b + 1) / nb) / 32);
}

// Stage the instance parts (H, A's bits when A.a_in_smem, unranking tables) into shared memory and
// zero cnt[]; returns A's bit rows. No barrier: callers follow with one.
template <int K>
__device__ const uint32_t *load_common(const SearchArgs &A, unsigned char *sm, const Smem &L)
{
    int *Hs = (int *)(sm + L.H);
    int *cnt = (int *)(sm + L.cnt);
    int *cur = (int *)(sm + L.cur);
    for (int b = threadIdx.x; b <= A.I.n; b += NT) Hs[b] = A.I.H[b];
    for (int u = threadIdx.x; u < A.I.n + 2 + 2 * K; u += NT) { cnt[u] = 0; cur[u] = 0; }
    fill_tables((uint32_t *)(sm + L.T2), (uint32_t *)(sm + L.T3), A.I.n);
    const uint32_t *Ar = A.I.Arow;
    if (A.a_in_smem) {
        uint32_t *As = (uint32_t *)(sm + L.Ar);
        const int nw = A.I.m * A.I.NWn;
        for (int q = threadIdx.x; q < nw; q += NT) As[q] = __ldg(A.I.Arow + q);
        Ar = As;
    }
    return Ar;
}

// Start a restart inside the CTA: V bits from the int8 vector V0, Y = A V0 (<a_j, v> = n - 2
// popcount(a xor v)), the range of Y, and f from scratch into ps.fpen/fhd:
// f = 30 fpen + fhd. Uses cur[] (n+1 zeroed entries) as the histogram and leaves it zeroed.
template <int K>
__device__ void init_restart(const SearchArgs &A, const uint32_t *Ar, const int8_t *V0, unsigned char *sm,
                             const Smem &L, PlanScalars &ps)
{
    int *Ys = (int *)(sm + L.Y);
    uint32_t *vbs = (uint32_t *)(sm + L.vb);
    const int *Hs = (const int *)(sm + L.H);
    int *hist = (int *)(sm + L.cur);
    for (int w = threadIdx.x; w < A.I.NWn; w += NT) vbs[w] = 0u;
    for (int b = threadIdx.x; b <= A.I.n; b += NT) hist[b] = 0;  // cur[] holds the last plan's cursors
    if (threadIdx.x == 0) { ps.fpen = 0; ps.fhd = 0; }
    __syncthreads();
    for (int i = threadIdx.x; i < A.I.n; i += NT)
        if (V0[i] < 0) atomicOr(&vbs[i >> 5], 1u << (i & 31));
    __syncthreads();
    int mn = INT_MAX, mx = INT_MIN, pen = 0;
    for (int j = threadIdx.x; j < A.I.m; j += NT) {
        const uint32_t *ar = Ar + (size_t)j * A.I.NWn;
        int d = 0;
        for (int w = 0; w < A.I.NWn; w++) d += __popc(ar[w] ^ vbs[w]);
        const int y = A.I.n - 2 * d;
        Ys[j] = y;
        mn = min(mn, y); mx = max(mx, y);
        if (y < 0) pen += -2 * y;
        else atomicAdd(&hist[y], 1);
    }
    atomicAdd(&ps.fpen, pen);
    range_publish<K>(mn, mx, ps);  // includes a __syncthreads: the histogram is complete
    int hd = 0;
    for (int b = threadIdx.x; b <= A.I.n; b += NT) { hd += abs(Hs[b] - hist[b]); hist[b] = 0; }
    atomicAdd(&ps.fhd, hd);
    __syncthreads();
}

// Stage the state (vb, Y) of a single search into shared memory and publish the range of Y.
template <int K>
__device__ const uint32_t *load_state(const SearchArgs &A, unsigned char *sm, const Smem &L, PlanScalars &ps)
{
    int *Ys = (int *)(sm + L.Y);
    uint32_t *vbs = (uint32_t *)(sm + L.vb);
    const uint32_t *Ar = load_common<K>(A, sm, L);
    int mn = INT_MAX, mx = INT_MIN;
    for (int j = threadIdx.x; j < A.I.m; j += NT) {
        const int y = A.Y[j];
        Ys[j] = y;
        mn = min(mn, y); mx = max(mx, y);
    }
    for (int w = threadIdx.x; w < A.I.NWn; w += NT) vbs[w] = A.vb[w];
    range_publish<K>(mn, mx, ps);
    __syncthreads();
    return Ar;
}

// Variant R3' (LNS_TABU_SOLUTIONS; PAPER.md:243-244 read literally, "the tabu list contains the
// solutions that have been visited in the recent past"): at iteration t the list holds
// V_{t-L} .. V_{t-1}. A neighbour V xor F equals a listed W iff F = V xor W, i.e. iff W differs
// from V in exactly k positions, and then F is those positions: each listed W marks at most one
// rank. The group's CTAs share the list (ring slot s mod L holds V_s); every CTA scans a strided
// share of it against vbs = V_{t-1} and writes until[rank] = t for the ranks of this device's
// slice (tabu at t, admissible again at t + 1: nothing to clear). CTA 0 stores V_{t-1} into its
// slot first (it is not among the listed entries scanned at t). A group barrier (arrival counter
// bar, monotonic, nb arrivals per pass; tb = this pass's number, one pass per iteration of the
// group) then publishes until[] before the evaluation reads it.
template <int K>
__device__ void sol_tabu(const SearchArgs &A, const unsigned char *sm, const Smem &L, const uint32_t *vbs,
                         int gg, uint32_t *until, int64_t t, int bid, int nb, unsigned long long *bar,
                         unsigned long long tb, int *xto)
{
    const int NW = A.I.NWn, n = A.I.n;
    const int64_t Lt = A.L;
    uint32_t *ring = A.ring + (size_t)gg * (size_t)Lt * NW;
    const uint32_t *T2 = (const uint32_t *)(sm + L.T2), *T3 = (const uint32_t *)(sm + L.T3);
    __syncthreads();  // vbs = V_{t-1}: the previous move was applied by the plan
    const int64_t skip = (t - 1) % Lt;  // slot of V_{t-1} (held V_{t-1-L}, no longer listed)
    if (bid == 0)
        for (int w = threadIdx.x; w < NW; w += NT) ring[(size_t)skip * NW + w] = vbs[w];
    // listed besides V_{t-1}: V_s, max(0, t-L) <= s <= t-2, i.e. every slot but `skip` once the
    // ring has wrapped, else slots 0 .. t-2
    const int64_t nlisted = min(t - 1, Lt - 1);
    for (int64_t j = (int64_t)bid * NT + threadIdx.x; j < nlisted; j += (int64_t)nb * NT) {
        const uint32_t *w = ring + (size_t)(j < skip ? j : j + 1) * NW;
        int d = 0;
        for (int q = 0; q < NW; q++) d += __popc(__ldcg(w + q) ^ vbs[q]);
        if (d != K) continue;
        int f[3] = {0, 0, 0}, cnt = 0;
        for (int q = 0; q < NW && cnt < K; q++)
            for (uint32_t x = __ldcg(w + q) ^ vbs[q]; x && cnt < K; x &= x - 1) f[cnt++] = 32 * q + __ffs(x) - 1;
        uint32_t r;
        if (K == 1) r = (uint32_t)f[0];
        else if (K == 2) r = A.M - 1u - (T2[n - 1 - f[0]] + (uint32_t)(n - 1 - f[1]));
        else r = A.M - 1u - (T3[n - 1 - f[0]] + T2[n - 1 - f[1]] + (uint32_t)(n - 1 - f[2]));
        if (r >= A.lo && r < A.hi) until[r] = (uint32_t)t;
    }
    if (nb > 1) {
        __syncthreads();
        if (threadIdx.x == 0) {
            __threadfence();
            asm volatile("red.release.gpu.global.add.u64 [%0], 1;" ::"l"(bar) : "memory");
            if (!spin_until_ge(bar, (unsigned long long)nb * tb, A.grid_timeout_ns)) *xto = 2;
            __threadfence();
        }
    }
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
    __shared__ int s_bad, s_hd;
    __shared__ unsigned long long s_pen;
    const int tid = threadIdx.x;
    if (tid == 0) { s_bad = 0; s_pen = 0; s_hd = 0; }
    for (int b = tid; b <= I.n; b += NT) hist[b] = 0;
    __syncthreads();
    for (int w = tid; w < I.NWn; w += NT) {
        uint32_t word = 0;
        for (int q = 0; q < 32; q++) {
            const int i = 32 * w + q;
            if (i < I.n) {
                const int8_t v = V0[i];
                if (v != 1 && v != -1) s_bad = 1;
                if (v < 0) word |= 1u << q;
            }
        }
        vb[w] = word;
    }
    __syncthreads();
    unsigned long long pen = 0;
    for (int j = tid; j < I.m; j += NT) {
        const uint32_t *ar = I.Arow + (size_t)j * I.NWn;
        int d = 0;
        for (int w = 0; w < I.NWn; w++) d += __popc(__ldg(ar + w) ^ vb[w]);
        const int y = I.n - 2 * d;  // <a_j, v> = n - 2 popcount(a xor v)
        Y[j] = y;
        if (Ycheck && Ycheck[j] != y) s_bad = 1;
        if (y < 0) pen += (unsigned long long)(-2 * y);
        if (y >= 0) atomicAdd(&hist[y], 1);
    }
    atomicAdd(&s_pen, pen);
    __syncthreads();
    int hd = 0;
    for (int b = tid; b <= I.n; b += NT) hd += abs(I.H[b] - hist[b]);
    atomicAdd(&s_hd, hd);
    __syncthreads();
    if (tid == 0) {
        const int64_t f = 30 * (int64_t)s_pen + s_hd;
        fs[FS_F] = f; fs[FS_T] = 0; fs[FS_BEST] = f; fs[FS_BESTIT] = 0;
        fs[FS_ZERO] = (f == 0) ? 0 : -1; fs[FS_DONE] = 0; fs[FS_ERR] = s_bad ? 1 : 0;
    }
}

// The persistent tabu search: all iterations in one cooperative launch. BATCH (A.R > 0): the grid
// is split into groups; each group runs its restarts one after another (batched restarts). The two
// modes are separate instantiations, so code that only one of them runs (the peer exchange and the
// flip-set keys of a single search) does not weigh on the other's register allocation.
template <int K, bool BATCH>
__global__ void __launch_bounds__(NT, 1) k_search(SearchArgs A)
{
    extern __shared__ __align__(16) unsigned char sm[];
    __shared__ PlanScalars ps;
    const Smem L = smem_layout(A.I.m, A.I.n, A.I.XW, A.I.NWn, K, A.a_in_smem, A.Xg != nullptr, A.I.pkw);
    int *Ys = (int *)(sm + L.Y);
    uint32_t *vbs = (uint32_t *)(sm + L.vb);
    constexpr bool batch = BATCH;
    const int lane = threadIdx.x & 31;
    const uint32_t *Ar = batch ? load_common<K>(A, sm, L) : load_state<K>(A, sm, L, ps);
    __shared__ unsigned long long *s_peers[MAX_PEERS];
    __shared__ int s_xto;
    if (threadIdx.x < A.npeers) s_peers[threadIdx.x] = A.peers[threadIdx.x];
    if (threadIdx.x == 0) s_xto = 0;
    __syncthreads();
#ifdef LNS_PHASE_TIMING
    if (threadIdx.x == 0) { for (int i = 0; i < NPH; i++) s_ph[i] = 0; s_last = clock64(); }
#endif
    for (int phq = 0; phq < (batch ? A.nph : 1); phq++) {
    const int G = batch ? A.phG[phq] : 1;
    const int nb = batch ? A.phnb[phq] : (int)gridDim.x;
    const int g = (int)blockIdx.x / nb, bid = (int)blockIdx.x - g * nb;
    if (g >= G) continue;  // idle in this phase
    const int gg = batch ? A.phgb[phq] + g : 0;  // global group index: exchange slots, until[]
    const bool leader = (bid == 0 && threadIdx.x == 0);
    unsigned long long *gslots = (unsigned long long *)A.slots + 64 * (size_t)gg;
    uint32_t blo, bhi;
    cta_slice(A.lo, A.hi, bid, nb, blo, bhi);
    // the CTA's until[] slice: shared-memory copy when it fits, else the group's global array, or
    // (bits_mode) the group's bitmap + ring of accepted ranks
    uint32_t *until = A.bits_mode ? nullptr : A.until + (batch ? (size_t)gg * A.M : 0);
    uint32_t *tb = A.bits_mode ? A.tbits + (size_t)gg * A.bit_words : nullptr;
    uint32_t *tring = (A.bits_mode && A.ring_on) ? A.tring + (size_t)gg * (size_t)A.L : nullptr;
    uint32_t ubase = 0;
    if (A.until_smem) {
        uint32_t *us = (uint32_t *)(sm + L.a_end);
        if (!batch)  // a new search: nothing is tabu
            for (uint32_t r = blo + threadIdx.x; r < bhi; r += NT) us[r - blo] = 0u;
        until = us;
        ubase = blo;
    }
    const uint2 *tri = nullptr;
    if (A.tri_smem) {
        uint2 *ts = (uint2 *)(sm + L.a_end + 4 * A.slice_cap);
        const uint32_t *T2 = (const uint32_t *)(sm + L.T2), *T3 = (const uint32_t *)(sm + L.T3);
        __syncthreads();  // the previous phase's readers of the table are done
        for (uint32_t r = blo + threadIdx.x; r < bhi; r += NT) {
            int a, b, c;
            unrank_tab<K>(r, A.I.n, A.M, T2, T3, a, b, c);
            ts[r - blo] = make_uint2((uint32_t)(a & 0xffff) | ((uint32_t)(b & 0xffff) << 16), (uint32_t)c);
        }
        __syncthreads();
        tri = ts;
    }
    unsigned long long tg = 0;  // iterations run by this group in this phase (exchange clock)
    const int rbeg = batch ? A.phr0[phq] : 0, rend = batch ? A.phr0[phq] + A.phR[phq] : 1;
    for (int rs = rbeg + (batch ? g : 0); rs < rend; rs += G) {
        int64_t f, best_f, best_it, zero_it, t0;
        if (batch) {
            init_restart<K>(A, Ar, A.V0s + (size_t)rs * A.I.n, sm, L, ps);
            if (tb)  // this CTA's words of the bitmap (slices are 32-aligned: no word is shared)
                for (uint32_t w = (blo >> 5) + threadIdx.x; w < ((bhi + 31) >> 5); w += NT) tb[w] = 0u;
            else
                for (uint32_t r = blo + threadIdx.x; r < bhi; r += NT) until[r - ubase] = 0u;
            __syncthreads();
            f = 30 * (int64_t)ps.fpen + ps.fhd;
            best_f = f; best_it = 0; zero_it = (f == 0) ? 0 : -1; t0 = 0;
        } else {
            f = A.fs[FS_F];
            best_f = A.fs[FS_BEST]; best_it = A.fs[FS_BESTIT]; zero_it = A.fs[FS_ZERO];
            t0 = A.fs[FS_T];
        }
        int64_t t = t0 + 1;
        bool failed = false;
        Move mv{0, 0, 0, 0};  // accepted, not yet applied
        for (; t <= t0 + A.iters; t++) {
            if (A.stop_on_zero && f == 0) break;
            if (A.Xg) build_plan<K, true, !BATCH>(A.I, Ar, sm, L, ps, X_OF(A, sm, L), mv);
            else build_plan<K, false, !BATCH>(A.I, Ar, sm, L, ps, nullptr, mv);
            // (the solution-list barrier is passed once per iteration, before the exchange: pass tg + 1)
            if (A.sol_list) {
                sol_tabu<K>(A, sm, L, vbs, gg, until, t, bid, nb, gslots + 24, tg + 1, &s_xto);
                if (s_xto) { failed = true; break; }
            }
            unsigned long long mine =
                A.Xg ? eval_range<K, false, true>(A.I, sm, L, ps, X_OF(A, sm, L), A.M, blo, bhi, until, ubase, (uint32_t)t,
                                                  nullptr, tri, A.aspiration, (int)best_f, tb, !BATCH && A.enc_keys)
                     : eval_range<K, false, false>(A.I, sm, L, ps, nullptr, A.M, blo, bhi, until, ubase, (uint32_t)t,
                                                   nullptr, tri, A.aspiration, (int)best_f, tb, !BATCH && A.enc_keys);
            mine = warp_min_k(mine);
            if (lane == 0 && mine != (unsigned long long)KEY_NONE) atomicMin(&ps.key, mine);
            // the rank leaving the FIFO after this iteration (accepted at t - L), read before this
            // CTA's arrival at exchange t; the leader overwrites its ring slot only after exchange t
            uint32_t evict = 0xffffffffu;
            if (tring && threadIdx.x == 0 && t > A.L) evict = __ldcg(tring + (size_t)((t - 1) % A.L));
            __syncthreads();
            PH(4);
            unsigned long long key = ps.key;
            tg++;
            if (!BATCH && A.npeers > 0) {
                // cross-GPU exchange (lns_attach_peers), two levels:
                //  1. inside the partition as below (.gpu scope): MIN into the local slot tg%3, one
                //     arrival on the local counter;
                //  2. CTA 0 waits for the local arrivals, MINs the partition's key into slot tg%3 of
                //     EVERY partition's exchange buffer and arrives on every partition's counter
                //     (.sys scope, NVLink peer memory), waits until its own counter shows all
                //     partitions, and reads its own slot: the global minimum;
                //  3. CTA 0 writes that key into the local slot and releases the local flag = tg;
                //     the other CTAs wait for the flag and read the slot.
                // Local slot (tg+2)%3 is reset by CTA 0 after the local arrivals at tg (its readers
                // read it at tg-1, before arriving at tg); its next writers pass the flag of tg+1,
                // which CTA 0 releases after the reset. The same holds per exchange buffer.
                if (threadIdx.x == 0) {
                    const int s3 = (int)(tg % 3);
                    unsigned long long *slot = gslots + 16 * s3;
                    unsigned long long *ctr = gslots + 48, *flag = gslots + 56;
                    if (key != (unsigned long long)KEY_NONE)
                        asm volatile("red.relaxed.gpu.global.min.u64 [%0], %1;" ::"l"(slot), "l"(key) : "memory");
                    asm volatile("red.release.gpu.global.add.u64 [%0], 1;" ::"l"(ctr) : "memory");
                    unsigned long long t_start, t_now, seen;
                    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_start));
                    bool late = false;
                    if (bid == 0) {
                        const unsigned long long local_target = (unsigned long long)nb * tg;
                        for (;;) {
                            asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(seen) : "l"(ctr) : "memory");
                            if (seen >= local_target) break;
                            asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_now));
                            if ((long long)(t_now - t_start) > A.timeout_ns) { late = true; break; }
                        }
                        if (!late) {
                            unsigned long long lk;
                            asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(lk) : "l"(slot) : "memory");
                            asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(gslots + 16 * ((tg + 2) % 3)),
                                         "l"((unsigned long long)KEY_NONE) : "memory");
                            if (lk != (unsigned long long)KEY_NONE)
                                for (int q = 0; q < A.npeers; q++)
                                    asm volatile("red.relaxed.sys.global.min.u64 [%0], %1;" ::"l"(s_peers[q] + 16 * s3),
                                                 "l"(lk) : "memory");
                            for (int q = 0; q < A.npeers; q++)
                                asm volatile("red.release.sys.global.add.u64 [%0], 1;" ::"l"(s_peers[q] + 48) : "memory");
                            unsigned long long *own = s_peers[A.part];
                            const unsigned long long target = (unsigned long long)A.npeers * tg;
                            for (;;) {
                                asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(seen) : "l"(own + 48) : "memory");
                                if (seen >= target) break;
                                asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_now));
                                if ((long long)(t_now - t_start) > A.timeout_ns) { late = true; break; }
                            }
                            if (!late) {
                                unsigned long long gk;
                                asm volatile("ld.relaxed.sys.global.u64 %0, [%1];" : "=l"(gk) : "l"(own + 16 * s3) : "memory");
                                asm volatile("st.relaxed.sys.global.u64 [%0], %1;" ::"l"(own + 16 * ((tg + 2) % 3)),
                                             "l"((unsigned long long)KEY_NONE) : "memory");
                                ps.gkey = gk;
                                asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(slot), "l"(gk) : "memory");
                                asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(flag), "l"(tg) : "memory");
                            }
                        }
                    } else {
                        for (;;) {
                            asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(seen) : "l"(flag) : "memory");
                            if (seen >= tg) break;
                            asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_now));
                            if ((long long)(t_now - t_start) > A.timeout_ns) { late = true; break; }
                        }
                        if (!late) {
                            unsigned long long gk;
                            asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(gk) : "l"(slot) : "memory");
                            ps.gkey = gk;
                        }
                    }
                    if (late) { s_xto = 1; ps.gkey = (unsigned long long)KEY_NONE; }
                }
                __syncthreads();
                key = ps.gkey;
                if (s_xto) { failed = true; break; }
            } else if (nb > 1) {
                // exchange: u64 MIN of this CTA's key into slot tg%3 (each slot on its own 128-B
                // line), then one arrival on the group's monotonic 64-bit counter; when it reaches
                // nb * tg every CTA's MIN has landed and the slot holds the group minimum. Slot
                // (tg+2)%3 was last read one exchange earlier by CTAs that have all arrived now,
                // so CTA 0 resets it here for exchange tg+2.
                if (threadIdx.x == 0) {
                    unsigned long long *slot = gslots + 16 * (tg % 3);
                    unsigned long long *ctr = gslots + 48;
                    if (key != (unsigned long long)KEY_NONE)
                        asm volatile("red.relaxed.gpu.global.min.u64 [%0], %1;" ::"l"(slot), "l"(key) : "memory");
                    // the release orders the MIN above before the arrival; the acquire below orders
                    // the slot read after every CTA's arrival (and hence its MIN)
                    asm volatile("red.release.gpu.global.add.u64 [%0], 1;" ::"l"(ctr) : "memory");
                    if (!spin_until_ge(ctr, (unsigned long long)nb * tg, A.grid_timeout_ns)) s_xto = 2;
                    unsigned long long gk;
                    asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(gk) : "l"(slot) : "memory");
                    ps.gkey = gk;
                    if (bid == 0)
                        asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(gslots + 16 * ((tg + 2) % 3)),
                                     "l"((unsigned long long)KEY_NONE) : "memory");
                }
                __syncthreads();
                key = ps.gkey;
                if (s_xto) { failed = true; break; }
            }
            PH(5);
            if (key == (unsigned long long)KEY_NONE) { failed = true; break; }
            // the accepted move: its flip set (the next plan applies it) and its rank
            uint32_t r;
            if (!BATCH && A.enc_keys) {
                dec_flip<K>((uint32_t)(key & 0xffffffffu), mv.a, mv.b, mv.c);
                r = rank_tab<K>(A.I.n, A.M, (const uint32_t *)(sm + L.T2), (const uint32_t *)(sm + L.T3), mv.a, mv.b, mv.c);
            } else {
                r = (uint32_t)(key & 0xffffffffu);
                unrank_tab<K>(r, A.I.n, A.M, (const uint32_t *)(sm + L.T2), (const uint32_t *)(sm + L.T3), mv.a, mv.b, mv.c);
            }
            f = (int64_t)(key >> 32);
            if (tb) {
                // bits_mode: r_{t-L} leaves the tabu list, r_t enters it (owner CTA's thread 0: the
                // only writer of its slice's words; its threads read them after the next barrier)
                if (threadIdx.x == 0) {
                    if (evict >= blo && evict < bhi) tb[evict >> 5] &= ~(1u << (evict & 31));
                    if (A.L > 0 && r >= blo && r < bhi) tb[r >> 5] |= 1u << (r & 31);
                    if (tring && bid == 0) __stcg(tring + (size_t)((t - 1) % A.L), r);
                }
            } else if (!A.sol_list && threadIdx.x == 0 && r >= blo && r < bhi) {
                until[r - ubase] = (uint32_t)(t + A.L);
            }
            if (leader) {
                if (A.trace_r) A.trace_r[t - 1] = r;
                if (A.trace_f) A.trace_f[t - 1] = f;
            }
            if (f < best_f) { best_f = f; best_it = t; }  // every thread (aspiration needs it)
            if (f == 0 && zero_it < 0) zero_it = t;
            // the move is applied by the next plan's step A (or below, after the last iteration)
            mv.on = 1;
            PH(6);
        }
        if (mv.on) apply_move<K>(A.I, Ar, Ys, vbs, mv.a, mv.b, mv.c);
        __syncthreads();  // the last move's V flip (thread 0) before V is written out / reused
        if (batch) {
            if (bid == 0) {
                for (int w = threadIdx.x; w < A.I.NWn; w += NT) A.vouts[(size_t)rs * A.I.NWn + w] = vbs[w];
                if (threadIdx.x == 0) {
                    int64_t *o = A.res + (size_t)rs * FS_N;
                    o[FS_F] = f; o[FS_T] = t - 1; o[FS_BEST] = best_f; o[FS_BESTIT] = best_it;
                    o[FS_ZERO] = zero_it; o[FS_DONE] = (A.stop_on_zero && f == 0) ? 1 : 0;
                    o[FS_ERR] = failed ? (s_xto == 2 ? 4 : 2) : 0;
                }
            }
        } else {
            if (bid == 0) {
                for (int j = threadIdx.x; j < A.I.m; j += NT) A.Y[j] = Ys[j];
                for (int w = threadIdx.x; w < A.I.NWn; w += NT) A.vb[w] = vbs[w];
                if (threadIdx.x == 0) {
                    A.fs[FS_F] = f; A.fs[FS_T] = t - 1; A.fs[FS_BEST] = best_f; A.fs[FS_BESTIT] = best_it;
                    A.fs[FS_ZERO] = zero_it; A.fs[FS_DONE] = (A.stop_on_zero && f == 0) ? 1 : 0;
                    if (failed) A.fs[FS_ERR] = s_xto == 2 ? 4 : s_xto ? 3 : 2;
                }
            }
        }
    }
    }  // phases
#ifdef LNS_PHASE_TIMING
    if (threadIdx.x == 0)
        for (int i = 0; i < NPH; i++) atomicAdd(&g_ph[i], (unsigned long long)s_ph[i]);
#endif
}

// Stepped mode, evaluation of iteration t = fs[FS_T] + 1: partial best key of this device's slice
// into key_out[0]. The last CTA to finish publishes the accumulator and resets it (no extra launch).
template <int K, bool WRITE_ALL>
__global__ void __launch_bounds__(NT, 1) k_step_eval(SearchArgs A, int64_t *key_out, int32_t *fit_out)
{
    extern __shared__ __align__(16) unsigned char sm[];
    __shared__ PlanScalars ps;
    const Smem L = smem_layout(A.I.m, A.I.n, A.I.XW, A.I.NWn, K, A.a_in_smem, A.Xg != nullptr, A.I.pkw);
    const int lane = threadIdx.x & 31;
    if (!WRITE_ALL && A.fs[FS_DONE]) {
        if (blockIdx.x == 0 && threadIdx.x == 0) *key_out = KEY_NONE;
        return;
    }
    const uint32_t *Ar = load_state<K>(A, sm, L, ps);
    uint32_t blo, bhi;
    cta_slice(A.lo, A.hi, blockIdx.x, gridDim.x, blo, bhi);
    if (A.Xg) build_plan<K, true>(A.I, Ar, sm, L, ps, X_OF(A, sm, L));
            else build_plan<K, false>(A.I, Ar, sm, L, ps, nullptr);
    const uint32_t t = (uint32_t)(A.fs[FS_T] + 1);
    unsigned long long mine =
        A.Xg ? eval_range<K, WRITE_ALL, true>(A.I, sm, L, ps, X_OF(A, sm, L), A.M, blo, bhi, A.until, 0, t, fit_out,
                                              nullptr, A.aspiration, (int)A.fs[FS_BEST])
             : eval_range<K, WRITE_ALL, false>(A.I, sm, L, ps, nullptr, A.M, blo, bhi, A.until, 0, t, fit_out,
                                               nullptr, A.aspiration, (int)A.fs[FS_BEST]);
    mine = warp_min_k(mine);
    if (lane == 0 && mine != (unsigned long long)KEY_NONE) atomicMin(&ps.key, mine);
    __syncthreads();
    if (threadIdx.x == 0) {
        if (ps.key != (unsigned long long)KEY_NONE) atomicMin((unsigned long long *)A.slots, ps.key);
        __threadfence();
        const unsigned done = atomicAdd(A.counter, 1u);
        if (done == gridDim.x - 1) {
            __threadfence();
            *key_out = (int64_t)atomicExch((unsigned long long *)A.slots, (unsigned long long)KEY_NONE);
            *A.counter = 0;
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
        if (r >= A.lo && r < A.hi) A.until[r] = (uint32_t)(t + A.L);
        if (A.trace_r) A.trace_r[t - 1] = r;
        if (A.trace_f) A.trace_f[t - 1] = f;
        A.fs[FS_F] = f; A.fs[FS_T] = t;
        if (f < A.fs[FS_BEST]) { A.fs[FS_BEST] = f; A.fs[FS_BESTIT] = t; }
        if (f == 0 && A.fs[FS_ZERO] < 0) A.fs[FS_ZERO] = t;
        if ((A.stop_on_zero && f == 0) || t >= A.iters) A.fs[FS_DONE] = 1;
    }
}

// Debug: dump the plan of the current state (one CTA):
// [vmin, U, NB, P, seg[0..U], bins (NB x {H, w}), pieces (P x {mask, meta}), pstart[0..W]]
template <int K>
__global__ void __launch_bounds__(NT, 1) k_debug_plan(SearchArgs A, int32_t *out)
{
    extern __shared__ __align__(16) unsigned char sm[];
    __shared__ PlanScalars ps;
    const Smem L = smem_layout(A.I.m, A.I.n, A.I.XW, A.I.NWn, K, A.a_in_smem, A.Xg != nullptr, A.I.pkw);
    const uint32_t *Ar = load_state<K>(A, sm, L, ps);
    const int *segp = (const int *)(sm + L.seg);
    if (A.Xg) build_plan<K, true>(A.I, Ar, sm, L, ps, X_OF(A, sm, L));
            else build_plan<K, false>(A.I, Ar, sm, L, ps, nullptr);
    const int U = ps.U;
    if (threadIdx.x == 0) {
        const int2 *bins = (const int2 *)(sm + L.bins);
        const uint2 *pieces = (const uint2 *)(sm + L.pieces);
        const int *pstart = (const int *)(sm + L.pstart);
        int o = 0;
        out[o++] = ps.vmin; out[o++] = U; out[o++] = ps.NB; out[o++] = ps.P;
        for (int u = 0; u <= U; u++) out[o++] = segp[u];
        for (int q = 0; q < ps.NB; q++) { out[o++] = bins[q].x; out[o++] = bins[q].y; }
        for (int q = 0; q < ps.P; q++) { out[o++] = (int)pieces[q].x; out[o++] = (int)pieces[q].y; }
        for (int w = 0; w <= ps.Wp; w++) out[o++] = pstart[w];
    }
}

// Unranking as the hot path does it (shared tables); tab = 0 uses the 64-bit reference version.
template <int K>
__global__ void k_unrank(int n, uint32_t M, const int64_t *ranks, int64_t count, int32_t *out, int32_t *bad, int tab)
{
    extern __shared__ uint32_t tabs[];
    uint32_t *T2 = tabs, *T3 = tabs + n;
    fill_tables(T2, T3, n);
    __syncthreads();
    for (int64_t q = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; q < count; q += (int64_t)gridDim.x * blockDim.x) {
        const int64_t r = ranks[q];
        if (r < 0 || r >= (int64_t)M) { *bad = 1; out[3 * q] = out[3 * q + 1] = out[3 * q + 2] = -1; continue; }
        int a, b, c;
        if (tab) unrank_tab<K>((uint32_t)r, n, M, T2, T3, a, b, c);
        else unrank<K>((uint32_t)r, n, M, a, b, c);
        out[3 * q] = a; out[3 * q + 1] = b; out[3 * q + 2] = c;
    }
}

__global__ void k_fill_i64(int64_t *p, int64_t v, int64_t cnt)
{
    for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < cnt; i += (int64_t)gridDim.x * blockDim.x) p[i] = v;
}

// Exchange slots of G groups: 3 keys (one per 128-B line) = KEY_NONE, arrival counter = 0.
__global__ void k_init_slots(int64_t *slots, int G)
{
    for (int i = blockIdx.x * blockDim.x + threadIdx.x; i < 64 * G; i += gridDim.x * blockDim.x) {
        const int q = i & 63;
        slots[i] = (q < 48 && q != 24) ? KEY_NONE : 0;  // q = 24: solution-list barrier counter
    }
}

// until[r] = bit r of the caller's tabu bitmap (tabu at t = 1 <=> until >= 1).
__global__ void k_bits_to_until(const uint32_t *bits, uint32_t *until, uint32_t M)
{
    for (uint32_t r = blockIdx.x * blockDim.x + threadIdx.x; r < M; r += gridDim.x * blockDim.x)
        until[r] = bits ? (bits[r >> 5] >> (r & 31)) & 1u : 0u;
}

// ------------------------------------------------------------------------------------------
// k = 4..7 ("k > 3 via the combinatorial number system"), m <= 255.
// A compact variant of the same method: exact combinatorial unranking for any k (the complement
// identity lex_rank(i_1 < .. < i_k) = M - 1 - sum_j C(n-1-i_j, k-j+1), u64 tables, binary
// search per position), lexicographic successor stepping over each thread's contiguous run of
// ranks, and the parity walks of §5.9 over (point, row word) pieces: the k columns of a row word
// are summed into three bit planes of t = #{i in F : x_ji = 1}, and a piece adds
// sum_rows 256^t (k masked plane-product POPCs) to a 64-bit window (bins u, u+2, .., u+2k of its
// walk: k+1 <= 8 bytes, counts <= m <= 255); when a point's last piece is done its bin (byte 0)
// is complete: f += w_b h + |h - H_b|, and the window shifts by one byte. Deep rows (Y < -2k) cost 60(2k - Y) - 240 t, rows above max(S) + 2k cost 1,
// bins of [0, n] outside both walks cost H_b. One persistent cooperative kernel per search, the
// same (f << 32 | r) key, warp/CTA argmin and counter exchange as k_search.
// ------------------------------------------------------------------------------------------
constexpr int KG_MAX = 7;
constexpr int NTG = 512;  // threads per CTA of the generic-k kernel (k registers of indices/masks)
#ifndef KGEN_OCC
#define KGEN_OCC 2  // CTAs per SM (64 registers per thread): 2 hide latency better than 1 (+20%)
#endif

struct GenArgs {
    DevInst I;
    int32_t K;
    uint32_t M;
    int64_t iters, L;
    int32_t stop_on_zero, aspiration;
    uint32_t *vb;
    int32_t *Y;
    int64_t *fs;
    uint32_t *until;
    int64_t *slots;
    int64_t *trace_r, *trace_f;
    int32_t *fit_out;  // non-null: write every rank's fitness (lns_eval_all), no search
    unsigned long long *best_out;  // non-null: MIN of the admissible keys (until[r] = 0) into it (eval_neighborhood)
    // batched restarts (R > 0): G groups of nbg CTAs; until[] of M entries and 64 exchange slots
    // per group; restart r from V0s + r n, results into res + r FS_N and vouts + r NWn
    int32_t R, G, nbg;
    int64_t grid_timeout_ns;  // give-up time of the in-kernel group exchange (then: no admissible move)
    const int8_t *V0s;
    int64_t *res;
    uint32_t *vouts;
};

struct GenSmem {
    int Bs, Y, vb, cnt, pos, cur, bins, C, X, pc, end;
};

__host__ __device__ inline GenSmem gen_layout(int m, int n, int NWn, int K)
{
    GenSmem s;
    int o = 0;
    s.Bs = o;   o = align16(o + 4 * m * NWn);          // sorted rows' sign bits x_jc
    s.Y = o;    o = align16(o + 4 * m);
    s.vb = o;   o = align16(o + 4 * NWn);
    s.cnt = o;  o = align16(o + 4 * (n + 1));           // rows per lattice point u = (Y + n) / 2
    s.pos = o;  o = align16(o + 4 * (n + 1));           // first sorted slot of point u
    s.cur = o;  o = align16(o + 4 * (n + 1));
    s.bins = o; o = align16(o + 8 * (n + 2 * K + 1));   // (H_b, w_b) of bin u' in [-K, n + K]
    s.C = o;    o = align16(o + 8 * (n + 1) * (K + 1)); // C(x, e), x <= n, e <= K (u64)
    const int W = (m + 31) >> 5;
    s.X = o;    o = align16(o + 4 * W * n);             // X[w][c]: column c's bits of sorted rows 32w..
    s.pc = o;   o = align16(o + 8 * 2 * (n + 3 + 2 * W)); // pieces of both walks (uint2)
    s.end = o;
    return s;
}

struct GenScalars {
    int ua, np[2], ndeep, ntop, walk0[2];
    int pc0[2], pc1[2];  // pieces of walk q: [pc0[q], pc1[q])
    int cbase;  // m - (H of the walked bins) + 60 sum_deep (2K - Y) + #top rows
    unsigned long long key, gkey;
};

__device__ __forceinline__ void gen_unrank(uint32_t r, int n, int K, uint32_t M, const unsigned long long *C,
                                           int *idx)
{
    unsigned long long R = (unsigned long long)(M - 1u - r);
    int cprev = n;
#pragma unroll
    for (int j = 0; j < KG_MAX; j++) {
        if (j < K) {
            const int e = K - j;
            int lo = e - 1, hi = cprev - 1;  // largest c in [lo, hi] with C(c, e) <= R (C(e-1, e) = 0)
            while (lo < hi) {
                const int mid = (lo + hi + 1) >> 1;
                if (C[mid * (K + 1) + e] <= R) lo = mid; else hi = mid - 1;
            }
            R -= C[lo * (K + 1) + e];
            idx[j] = n - 1 - lo;
            cprev = lo;
        }
    }
}

// Lexicographic successor (the last index varies fastest; loops unrolled so idx stays in
// registers). Only called when a successor exists.
__device__ __forceinline__ void gen_succ(int n, int K, int *idx)
{
    int j = K - 1;  // rightmost index that can still advance
#pragma unroll
    for (int q = KG_MAX - 1; q > 0; q--)
        if (q == j && idx[q] == n - K + q) j--;
#pragma unroll
    for (int q = 0; q < KG_MAX; q++) {
        if (q == j) idx[q]++;
        else if (q > 0 && q > j && q < K) idx[q] = idx[q - 1] + 1;
    }
}

// Plan of the current (Y, V): apply the pending move first (pending = K indices, or none).
__device__ void gen_plan(const GenArgs &A, unsigned char *sm, const GenSmem &L, GenScalars &gs, const int *mvidx,
                         bool pending)
{
    const int tid = threadIdx.x, m = A.I.m, n = A.I.n, NWn = A.I.NWn, K = A.K;
    uint32_t *Bs = (uint32_t *)(sm + L.Bs);
    int *Ys = (int *)(sm + L.Y), *cnt = (int *)(sm + L.cnt), *pos = (int *)(sm + L.pos), *cur = (int *)(sm + L.cur);
    uint32_t *vbs = (uint32_t *)(sm + L.vb);
    int2 *bins = (int2 *)(sm + L.bins);
    const uint32_t *Ar = A.I.Arow;
    for (int u = tid; u <= n; u += NTG) cnt[u] = 0;
    if (pending) {  // Y'_j = Y_j - 2 sum_{i in F} B_ji = Y_j - 2K + 4 t_j
        for (int j = tid; j < m; j += NTG) {
            int t = 0;
            for (int q = 0; q < K; q++) {
                const int i = mvidx[q];
                t += (int)(((__ldg(Ar + (size_t)j * NWn + (i >> 5)) ^ vbs[i >> 5]) >> (i & 31)) & 1u);
            }
            Ys[j] += 4 * t - 2 * K;
        }
        __syncthreads();
        if (tid == 0)
            for (int q = 0; q < K; q++) vbs[mvidx[q] >> 5] ^= 1u << (mvidx[q] & 31);
    }
    __syncthreads();
    for (int j = tid; j < m; j += NTG) atomicAdd(&cnt[(Ys[j] + n) >> 1], 1);
    __syncthreads();
    if (tid == 0) {
        // walked points: -2K <= Y = 2u - n <= maxS + 2K; placement deep | walk 0 | walk 1 | top
        const int ua = max(0, (n - 2 * K + 1) >> 1), ub = min(n, (A.I.maxS + 2 * K + n) >> 1);
        int p = 0, cdeep = 0;
        for (int u = 0; u < min(ua, n + 1); u++) { pos[u] = p; p += cnt[u]; cdeep += cnt[u] * 60 * (2 * K - (2 * u - n)); }
        gs.ndeep = p;
        int hwalk = 0;
        for (int q = 0; q < 2; q++) {
            int np = 0;
            for (int u = ua + q; u <= ub; u += 2) { pos[u] = p; p += cnt[u]; np++; }
            gs.np[q] = np;
            gs.walk0[q] = ua + q;
            for (int P = 0; P < np + K; P++) {  // bins of walk positions 0 .. np + K - 1
                const int b = 2 * (ua + q + 2 * P - K) - n;
                if (np > 0 && b >= 0 && b <= n) hwalk += A.I.H[b];
            }
        }
        const int pt = p;
        for (int u = max(ub + 1, ua); u <= n; u++) { pos[u] = p; p += cnt[u]; }
        gs.ntop = p - pt;
        gs.ua = ua;
        gs.cbase = m - hwalk + cdeep + gs.ntop;
        gs.key = (unsigned long long)KEY_NONE;
        gs.gkey = (unsigned long long)KEY_NONE;
    }
    for (int x = tid; x < n + 2 * K + 1; x += NTG) {
        const int b = 2 * (x - K) - n;
        bins[x] = make_int2((b >= 0 && b <= n) ? A.I.H[b] : 0, b < 0 ? 60 * (-b) - 1 : 0);
    }
    __syncthreads();
    for (int u = tid; u <= n; u += NTG) cur[u] = pos[u];
    __syncthreads();
    for (int j = tid; j < m; j += NTG) {
        const int p = atomicAdd(&cur[(Ys[j] + n) >> 1], 1);
        for (int w = 0; w < NWn; w++) Bs[p * NWn + w] = __ldg(Ar + (size_t)j * NWn + w) ^ vbs[w];
    }
    __syncthreads();
    // X[w][c] = column c's bits over sorted rows 32w .. 32w+31 (row-major Bs transposed), and the
    // pieces of each walk: (mask, word | last << 15 | popc(mask) << 16) per (point, row word), an
    // empty point one zero piece that only completes its bin
    uint32_t *X = (uint32_t *)(sm + L.X);
    const int W = (m + 31) >> 5;
    for (int e = tid; e < W * n; e += NTG) {
        const int w = e / n, c = e - w * n;
        uint32_t x = 0;
        for (int l = 0; l < 32 && 32 * w + l < m; l++)
            x |= ((Bs[(32 * w + l) * NWn + (c >> 5)] >> (c & 31)) & 1u) << l;
        X[e] = x;
    }
    if (tid == 0) {
        uint2 *pc = (uint2 *)(sm + L.pc);
        int np_ = 0;
        for (int q = 0; q < 2; q++) {
            gs.pc0[q] = np_;
            int lastw = 0;
            for (int P = 0; P < gs.np[q]; P++) {
                const int u = gs.walk0[q] + 2 * P, st = pos[u], en = st + cnt[u];
                if (en == st) { pc[np_++] = make_uint2(0u, (uint32_t)lastw | (1u << 15)); continue; }
                for (int w = st >> 5; w <= (en - 1) >> 5; w++) {
                    const int lo = max(st, 32 * w) - 32 * w, hi = min(en, 32 * w + 32) - 32 * w;
                    const uint32_t mask = (hi == 32 ? FULL : ((1u << hi) - 1u)) & (FULL << lo);
                    pc[np_++] = make_uint2(mask, (uint32_t)w | ((w == (en - 1) >> 5) ? 1u << 15 : 0u) |
                                                     ((uint32_t)__popc(mask) << 16));
                    lastw = w;
                }
            }
            gs.pc1[q] = np_;
        }
    }
    __syncthreads();
}

// Bit-sliced planes of t = #{i in F : x_i = 1} over one row word (t <= 7: three planes).
__device__ __forceinline__ void gen_planes(const uint32_t *__restrict__ xw, const int *idx, int K, uint32_t &b0,
                                           uint32_t &b1, uint32_t &b2)
{
    b0 = 0; b1 = 0; b2 = 0;
#pragma unroll
    for (int j = 0; j < KG_MAX; j++) {
        if (j < K) {
            const uint32_t x = xw[idx[j]];
            const uint32_t c0 = b0 & x;
            b0 ^= x;
            b2 |= b1 & c0;
            b1 ^= c0;
        }
    }
}

// Fitness of the neighbour idx[0..K) from the plan. Per piece (the rows of one lattice point in
// one row word, mask m) the walk window gains sum_rows 256^t = popc(m) + sum (256^t - 1), and with
// t = b0 + 2 b1 + 4 b2: 256^t - 1 = (1 + 255 b0)(1 + 65535 b1)(1 + (2^32 - 1) b2) - 1, i.e. seven
// masked plane products (those K cannot reach vanish: K = 4 needs 4 POPCs, 5: 5, 6: 6, 7: 7).
template <int KT>
__device__ __forceinline__ int gen_eval(const GenArgs &A, const unsigned char *sm, const GenSmem &L,
                                        const GenScalars &gs, const int *idx)
{
    constexpr int K = KT;
    const int n = A.I.n;
    const uint32_t *X = (const uint32_t *)(sm + L.X);
    const uint2 *pc = (const uint2 *)(sm + L.pc);
    const int2 *bins = (const int2 *)(sm + L.bins);
    int f = gs.cbase;
    uint32_t b0, b1, b2;
    for (int w = 0, nd = gs.ndeep; 32 * w < nd; w++) {  // deep rows: -240 sum t
        gen_planes(X + w * n, idx, K, b0, b1, b2);
        const uint32_t dm = (nd - 32 * w >= 32) ? FULL : ((1u << (nd - 32 * w)) - 1u);
        f -= 240 * (__popc(b0 & dm) + 2 * __popc(b1 & dm) + 4 * __popc(b2 & dm));
    }
    for (int q = 0; q < 2; q++) {
        if (gs.np[q] == 0) continue;
        unsigned long long win = 0;
        int curw = -1, u = gs.walk0[q];
        for (int e = gs.pc0[q]; e < gs.pc1[q]; e++) {
            const uint2 pr = pc[e];
            const int w = (int)(pr.y & 0x7fffu);
            if (w != curw) { gen_planes(X + w * n, idx, K, b0, b1, b2); curw = w; }
            const uint32_t m = pr.x;
            unsigned long long d = (unsigned long long)(pr.y >> 16);
            d += 255ull * __popc(b0 & m) + 65535ull * __popc(b1 & m) + 16711425ull * __popc(b0 & b1 & m);
            if (K >= 4) d += 4294967295ull * __popc(b2 & m);
            if (K >= 5) d += 1095216660225ull * __popc(b0 & b2 & m);     // 255 (2^32 - 1)
            if (K >= 6) d += 281470681677825ull * __popc(b1 & b2 & m);  // 65535 (2^32 - 1)
            if (K >= 7) d += 71775023827845375ull * __popc(b0 & b1 & b2 & m);  // 255 * 65535 (2^32 - 1)
            win += d;
            if (pr.y & (1u << 15)) {  // the point's last piece: its bin is complete
                const int h = (int)(win & 0xffu);
                const int2 bn = bins[u];  // bin u' = u - K, stored at u' + K = u
                f += bn.y * h + abs(h - bn.x);
                win >>= 8;
                u += 2;
            }
        }
        for (int P = 0; P < K; P++, u += 2) {  // trailing bins: rows carried past the last point
            const int h = (int)(win & 0xffu);
            const int2 bn = bins[u];
            f += bn.y * h + abs(h - bn.x);
            win >>= 8;
        }
    }
    return f;
}

// One instantiation per k (4..7): the plane loops and the product terms fold at compile time.
template <int KT>
__global__ void __launch_bounds__(NTG, KGEN_OCC) k_gen(GenArgs A)
{
    extern __shared__ __align__(16) unsigned char sm[];
    __shared__ GenScalars gs;
    __shared__ int s_mv[KG_MAX];
    __shared__ int s_pen, s_hd;
    const GenSmem L = gen_layout(A.I.m, A.I.n, A.I.NWn, A.K);
    constexpr int K = KT;
    const int tid = threadIdx.x, lane = tid & 31, n = A.I.n, m = A.I.m, NWn = A.I.NWn;
    // batched restarts (A.R > 0): group g = CTAs [g nbg, (g+1) nbg) runs restarts g, g + G, ...
    const bool batch = A.R > 0;
    const int nbg = batch ? A.nbg : (int)gridDim.x;
    const int g = (int)blockIdx.x / nbg, bid = (int)blockIdx.x - g * nbg;
    if (batch && g >= A.G) return;
    unsigned long long *C = (unsigned long long *)(sm + L.C);
    for (int x = tid; x <= n; x += NTG) {  // C(x, e) by Pascal's rule along e (exact in u64 here)
        unsigned long long c = 1;
        for (int e = 0; e <= K; e++) {
            C[x * (K + 1) + e] = (e <= x) ? c : 0ull;
            c = (e < x) ? c * (unsigned long long)(x - e) / (unsigned long long)(e + 1) : 0ull;
        }
    }
    int *Ys = (int *)(sm + L.Y);
    uint32_t *vbs = (uint32_t *)(sm + L.vb);
    if (!batch) {
        for (int j = tid; j < m; j += NTG) Ys[j] = A.Y[j];
        for (int w = tid; w < NWn; w += NTG) vbs[w] = A.vb[w];
    }
    __syncthreads();
    // this thread's contiguous run of ranks (within its group)
    const uint64_t span = A.M, gt = (uint64_t)bid * NTG + tid, Gt = (uint64_t)nbg * NTG;
    const uint32_t lo = (uint32_t)(span * gt / Gt), hi = (uint32_t)(span * (gt + 1) / Gt);
    if (A.fit_out || A.best_out) {
        gen_plan(A, sm, L, gs, s_mv, false);
        int idx[KG_MAX];
        unsigned long long best = (unsigned long long)KEY_NONE;
        if (lo < hi) gen_unrank(lo, n, K, A.M, C, idx);
        for (uint32_t r = lo; r < hi; r++) {
            if (A.fit_out) A.fit_out[r] = gen_eval<KT>(A, sm, L, gs, idx);
            else if (A.until[r] == 0u) {
                const unsigned long long key = ((unsigned long long)(uint32_t)gen_eval<KT>(A, sm, L, gs, idx) << 32) | r;
                if (key < best) best = key;
            }
            if (r + 1 < hi) gen_succ(n, K, idx);
        }
        if (A.best_out) {
            best = warp_min_k(best);
            if (lane == 0 && best != (unsigned long long)KEY_NONE) atomicMin(A.best_out, best);
        }
        return;
    }
    uint32_t *until = A.until + (batch ? (size_t)g * A.M : 0);
    unsigned long long *slots = (unsigned long long *)A.slots + 64 * (size_t)g;
    unsigned long long tg = 0;  // exchanges of this group (monotonic across its restarts)
    for (int rs = batch ? g : 0; rs < (batch ? A.R : 1); rs += (batch ? A.G : 1)) {
        int64_t f, best_f, best_it, zero_it, t0;
        if (batch) {
            // restart rs from V0s[rs]: V bits, Y = A V, f from scratch
            int *hist = (int *)(sm + L.cnt);
            for (int w = tid; w < NWn; w += NTG) vbs[w] = 0u;
            for (int b = tid; b <= n; b += NTG) hist[b] = 0;
            if (tid == 0) { s_pen = 0; s_hd = 0; }
            __syncthreads();
            const int8_t *V0 = A.V0s + (size_t)rs * n;
            for (int i = tid; i < n; i += NTG)
                if (V0[i] < 0) atomicOr(&vbs[i >> 5], 1u << (i & 31));
            __syncthreads();
            int pen = 0;
            for (int j = tid; j < m; j += NTG) {
                int d = 0;
                for (int w = 0; w < NWn; w++) d += __popc(__ldg(A.I.Arow + (size_t)j * NWn + w) ^ vbs[w]);
                const int y = n - 2 * d;
                Ys[j] = y;
                if (y < 0) pen += -2 * y;
                else atomicAdd(&hist[y], 1);
            }
            atomicAdd(&s_pen, pen);
            __syncthreads();
            int hd = 0;
            for (int b = tid; b <= n; b += NTG) hd += abs(A.I.H[b] - hist[b]);
            atomicAdd(&s_hd, hd);
            for (uint32_t r = lo; r < hi; r++) until[r] = 0u;  // this thread's ranks only
            __syncthreads();
            f = 30 * (int64_t)s_pen + s_hd;
            best_f = f; best_it = 0; zero_it = (f == 0) ? 0 : -1; t0 = 0;
        } else {
            f = A.fs[FS_F]; best_f = A.fs[FS_BEST]; best_it = A.fs[FS_BESTIT]; zero_it = A.fs[FS_ZERO];
            t0 = A.fs[FS_T];
        }
        int64_t t = t0 + 1;
        bool failed = false, pending = false;
        for (; t <= t0 + A.iters; t++) {
            if (A.stop_on_zero && f == 0) break;
            gen_plan(A, sm, L, gs, s_mv, pending);
            unsigned long long best = (unsigned long long)KEY_NONE;
            int idx[KG_MAX];
            if (lo < hi) gen_unrank(lo, n, K, A.M, C, idx);
            for (uint32_t r = lo; r < hi; r++) {
                const bool tabu = until[r] >= (uint32_t)t;
                if (!tabu || A.aspiration) {
                    const int fr = gen_eval<KT>(A, sm, L, gs, idx);
                    const unsigned long long key = ((unsigned long long)(uint32_t)fr << 32) | r;
                    if ((!tabu || fr < best_f) && key < best) best = key;
                }
                if (r + 1 < hi) gen_succ(n, K, idx);
            }
            best = warp_min_k(best);
            if (lane == 0 && best != (unsigned long long)KEY_NONE) atomicMin(&gs.key, best);
            __syncthreads();
            unsigned long long key = gs.key;
            tg++;
            if (nbg > 1) {  // the counter exchange of k_search, per group
                if (tid == 0) {
                    unsigned long long *slot = slots + 16 * (tg % 3), *ctr = slots + 48;
                    if (key != (unsigned long long)KEY_NONE)
                        asm volatile("red.relaxed.gpu.global.min.u64 [%0], %1;" ::"l"(slot), "l"(key) : "memory");
                    asm volatile("red.release.gpu.global.add.u64 [%0], 1;" ::"l"(ctr) : "memory");
                    unsigned long long gk;
                    if (!spin_until_ge(ctr, (unsigned long long)nbg * tg, A.grid_timeout_ns)) gk = KEY_NONE;
                    else asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(gk) : "l"(slot) : "memory");
                    gs.gkey = gk;
                    if (bid == 0)
                        asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(slots + 16 * ((tg + 2) % 3)),
                                     "l"((unsigned long long)KEY_NONE) : "memory");
                }
                __syncthreads();
                key = gs.gkey;
            }
            if (key == (unsigned long long)KEY_NONE) { failed = true; break; }
            const uint32_t r = (uint32_t)(key & 0xffffffffu);
            f = (int64_t)(key >> 32);
            // the owner of rank r (the thread whose run holds it) sets until[r]: exactly one writer
            if (r >= lo && r < hi) until[r] = (uint32_t)(t + A.L);
            if (!batch && bid == 0 && tid == 0) {
                if (A.trace_r) A.trace_r[t - 1] = r;
                if (A.trace_f) A.trace_f[t - 1] = f;
            }
            if (f < best_f) { best_f = f; best_it = t; }
            if (f == 0 && zero_it < 0) zero_it = t;
            if (tid == 0) {
                int mi[KG_MAX];
                gen_unrank(r, n, K, A.M, C, mi);
                for (int q = 0; q < K; q++) s_mv[q] = mi[q];
            }
            pending = true;
            __syncthreads();
        }
        if (pending) gen_plan(A, sm, L, gs, s_mv, true);  // applies the last move (Y, V)
        if (bid == 0) {
            if (batch) {
                for (int w = tid; w < NWn; w += NTG) A.vouts[(size_t)rs * NWn + w] = vbs[w];
                if (tid == 0) {
                    int64_t *o = A.res + (size_t)rs * FS_N;
                    o[FS_F] = f; o[FS_T] = t - 1; o[FS_BEST] = best_f; o[FS_BESTIT] = best_it;
                    o[FS_ZERO] = zero_it; o[FS_DONE] = (A.stop_on_zero && f == 0) ? 1 : 0;
                    o[FS_ERR] = failed ? 2 : 0;
                }
            } else {
                for (int j = tid; j < m; j += NTG) A.Y[j] = Ys[j];
                for (int w = tid; w < NWn; w += NTG) A.vb[w] = vbs[w];
                if (tid == 0) {
                    A.fs[FS_F] = f; A.fs[FS_T] = t - 1; A.fs[FS_BEST] = best_f; A.fs[FS_BESTIT] = best_it;
                    A.fs[FS_ZERO] = zero_it; A.fs[FS_DONE] = (A.stop_on_zero && f == 0) ? 1 : 0;
                    if (failed) A.fs[FS_ERR] = 2;
                }
            }
        }
        __syncthreads();  // vbs / Ys are reused by the next restart
    }
}

__global__ void k_unrank_gen(int n, int K, uint32_t M, const int64_t *ranks, int64_t count, int32_t *out, int32_t *bad)
{
    extern __shared__ __align__(16) unsigned char smc[];
    unsigned long long *C = (unsigned long long *)smc;
    for (int x = threadIdx.x; x <= n; x += blockDim.x) {
        unsigned long long c = 1;
        for (int e = 0; e <= K; e++) {
            C[x * (K + 1) + e] = (e <= x) ? c : 0ull;
            c = (e < x) ? c * (unsigned long long)(x - e) / (unsigned long long)(e + 1) : 0ull;
        }
    }
    __syncthreads();
    for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < count; i += (int64_t)gridDim.x * blockDim.x) {
        const int64_t r = ranks[i];
        if (r < 0 || r >= (int64_t)M) { *bad = 1; continue; }
        int idx[KG_MAX];
        gen_unrank((uint32_t)r, n, K, M, C, idx);
        for (int q = 0; q < K; q++) out[i * K + q] = idx[q];
    }
}

}  // namespace

// ==========================================================================================
// Host side
// ==========================================================================================
typedef int (*nccl_allreduce_fn)(const void *, void *, size_t, int, int, void *, cudaStream_t);

struct lns_ctx {
    int device = 0;
    int m = 0, n = 0, W = 0, NWn = 0, maxS = 0;
    uint32_t *d_Arow = nullptr;
    int32_t *d_H = nullptr;
    int numSMs = 0, smemOptin = 0;
    int part = 0, nparts = 1;
    void *comm = nullptr;
    nccl_allreduce_fn nccl_allreduce = nullptr;
    void *comm_owned = nullptr;       // created by lns_comm_init_rank (destroyed with the context)
    void *nccl_lib = nullptr;         // dl handle the communicator's NCCL calls come from
    int blocks_override = 0;
    int no_pad = 0;  // LNS_NO_PAD=1 at create: plain (unpadded) row placement, for A/B measurement
    int no_pkw = 0;  // LNS_NO_PKW=1 at create: m > 255 always takes the segment plan (A/B measurement)
    int force_pkw = 0;  // LNS_FORCE_PKW=1 at create: m > 255 tries the packed plan for any slice size
    int no_graph = 0;   // LNS_NO_GRAPH=1 at create: the stepped loop launches directly (A/B measurement)
    int64_t grid_timeout_ms = 60000;  // LNS_GRID_TIMEOUT_MS at create: give-up time of an in-kernel grid exchange
    cudaStream_t cap_stream = nullptr;  // private stream for capturing the stepped loop's graph
    // device-initiated exchange (lns_attach_peers)
    unsigned long long *d_xbuf = nullptr;            // own 64-word exchange buffer (its own allocation)
    unsigned long long **d_peers = nullptr;          // device array of the partitions' buffers
    int npeers = 0;
    int64_t peer_timeout_ms = 0;
    std::vector<void *> ipc_opened;                   // peer buffers opened by lns_attach_peers_ipc
    // run state
    uint32_t *d_vb = nullptr;
    int32_t *d_Y = nullptr;
    int64_t *d_fs = nullptr;
    int64_t *d_slots = nullptr;  // 3 x MAX_SLOTS persistent slots, then stepped accumulator, eval output
    unsigned *d_counter = nullptr;
    int8_t *d_V = nullptr;
    int32_t *d_Yin = nullptr;
    uint32_t *d_bits = nullptr; size_t bits_cap = 0;
    uint32_t *d_until = nullptr; size_t until_cap = 0;
    uint32_t *d_tbits = nullptr; size_t tbits_cap = 0;        // bits_mode tabu bitmaps (per group)
    uint32_t *d_tring = nullptr; size_t tring_cap = 0;        // bits_mode rings of accepted ranks
    int no_bits = 0;    // LNS_NO_BITS=1 at create: global until[] instead of bitmap + ring (A/B)
    int64_t *d_tr = nullptr, *d_tf = nullptr; size_t trace_cap = 0, trace_cap_f = 0;
    int32_t *d_fit = nullptr; size_t fit_cap = 0;
    int8_t *d_V0s = nullptr; size_t v0s_cap = 0;       // batched restarts
    int64_t *d_res = nullptr; size_t res_cap = 0;
    uint32_t *d_vouts = nullptr; size_t vouts_cap = 0;
    int64_t *d_gslots = nullptr; size_t gslots_cap = 0;
    uint32_t *d_X = nullptr; size_t X_cap = 0;                // global X fallback (per CTA)
    uint32_t *d_ring = nullptr; size_t ring_cap = 0;          // LNS_TABU_SOLUTIONS: visited solutions
    cudaEvent_t ev0 = nullptr, ev1 = nullptr;
    cudaEvent_t ev2 = nullptr, ev3 = nullptr;  // stepped loop: graph build excluded from last_ms
    double last_ms = 0.0;
    // stepped search
    bool step_active = false;
    int step_K = 0; int64_t step_iters = 0, step_L = 0; int step_flags = 0;
};

namespace {

constexpr int SLOT_ACC = 3 * MAX_SLOTS;  // stepped accumulator
constexpr int SLOT_OUT = 3 * MAX_SLOTS + 1;  // eval output key
constexpr int SLOT_N = 3 * MAX_SLOTS + 2;

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
    if (k < 1 || k > KG_MAX) return -1;
    if (n < k) return 0;
    int64_t c = 1;  // C(n, k) = prod_{i < k} (n - i) / (i + 1), exact at every step; capped
    for (int i = 0; i < k; i++) {
        c = c * (n - i) / (i + 1);
        if (c > ((int64_t)1 << 40)) return INT64_MAX;
    }
    return c;
}

DevInst dev_inst(const lns_ctx *c) { return DevInst{c->m, c->n, c->W, c->NWn, c->W, 0, c->d_Arow, c->d_H, c->maxS}; }

// Per-device caching allocator for context buffers (lns_pool_*). cudaMalloc / cudaFree cost tens
// of microseconds to milliseconds each and cudaFree synchronises the device, so a user who creates a
// context per instance (the e2e path: lns_create -> run -> lns_destroy) would pay them on every
// call. Freed blocks are kept per (device, power-of-two size class) and handed to the next request
// of that class; the cache is bounded (LNS_POOL_CAP_MB, default 4096) and lns_pool_trim() returns
// it to the driver. Every public call that launches work synchronises its stream before it
// returns, so a block is never recycled while a kernel still uses it (lns_destroy synchronises the
// device first when a stepped search is still open).
struct Pool {
    std::mutex mu;
    std::multimap<std::pair<int, size_t>, void *> cache;   // (device, class) -> free block
    std::map<void *, std::pair<int, size_t>> live;          // block -> (device, class)
    size_t cached = 0, live_bytes = 0, cap = 0;
};
Pool &pool()
{
    static Pool *p = [] {
        Pool *q = new Pool();  // never destroyed: no dependence on static teardown order
        const char *e = getenv("LNS_POOL_CAP_MB");
        q->cap = (size_t)(e ? atol(e) : 4096) << 20;
        return q;
    }();
    return *p;
}
size_t size_class(size_t b)
{
    size_t c = 256;
    while (c < b) c <<= 1;
    return c;
}
cudaError_t pool_alloc(void **out, size_t bytes)
{
    int dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return e;
    const size_t cls = size_class(bytes);
    Pool &P = pool();
    {
        std::lock_guard<std::mutex> lk(P.mu);
        auto it = P.cache.find({dev, cls});
        if (it != P.cache.end()) {
            *out = it->second;
            P.cache.erase(it);
            P.cached -= cls;
            P.live[*out] = {dev, cls};
            P.live_bytes += cls;
            return cudaSuccess;
        }
    }
    e = cudaMalloc(out, cls);
    if (e != cudaSuccess) {
        cudaGetLastError();
        lns_pool_trim();  // retry once with the cache released
        e = cudaMalloc(out, cls);
        if (e != cudaSuccess) { cudaGetLastError(); *out = nullptr; return e; }
    }
    std::lock_guard<std::mutex> lk(P.mu);
    P.live[*out] = {dev, cls};
    P.live_bytes += cls;
    return cudaSuccess;
}
template <typename T>
cudaError_t pool_alloc(T **out, size_t bytes) { return pool_alloc((void **)out, bytes); }
void pool_free(void *p)
{
    if (!p) return;
    Pool &P = pool();
    std::unique_lock<std::mutex> lk(P.mu);
    auto it = P.live.find(p);
    if (it == P.live.end()) return;  // not ours (never happens)
    const auto key = it->second;
    P.live.erase(it);
    P.live_bytes -= key.second;
    if (P.cached + key.second <= P.cap) {
        P.cache.insert({key, p});
        P.cached += key.second;
        return;
    }
    lk.unlock();
    int cur = 0;
    cudaGetDevice(&cur);
    if (cur != key.first) cudaSetDevice(key.first);
    cudaFree(p);
    if (cur != key.first) cudaSetDevice(cur);
}

template <typename T>
lns_status grow(T *&p, size_t &cap, size_t need)
{
    if (need <= cap && p) return LNS_OK;
    pool_free(p);
    p = nullptr; cap = 0;
    if (pool_alloc(&p, need * sizeof(T) + 16) != cudaSuccess) return fail(LNS_ENOMEM, "cudaMalloc failed");
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

// Launch geometry of one search: k, shared-memory bytes, A staged or not, until cached or not.
struct Geometry {
    uint32_t M = 0;
    int a_in_smem = 0;
    int x_global = 0;      // X does not fit in shared memory: per-CTA slots in global memory
    int pad = 0, XW = 0;   // padded placement (packed path, when X of 2W + 1 words fits)
    int pkw = 0;           // m > 255: packed records allocated, the packed plan tried per iteration
    int pkw_force = 0;     // LNS_FORCE_PKW=1 at create: try it for any slice size (tests)
    size_t smem_eval = 0;  // bytes for the stepped / eval kernels
};

// Shared-memory geometry of the plan for k (pkw: with the packed-record region for m > 255).
lns_status geometry(lns_ctx *c, int k, Geometry &g, int pkw)
{
    g.pkw = c->m > PACKED_MAX_M ? pkw : 0;
    g.a_in_smem = 0; g.x_global = 0; g.smem_eval = 0;
    const int budget = c->smemOptin - 1024;  // static shared memory of the kernels stays < 1 KiB
    // preference: X and A in shared memory; X only; neither (X in global memory)
    // padded placement first (packed path only): X of 2W + 1 words, with or without A staged
    g.pad = 0; g.XW = c->W;
    if (c->m <= PACKED_MAX_M && !c->no_pad) {
        const int XWp = 2 * c->W + 1;
        const Smem pw = smem_layout(c->m, c->n, XWp, c->NWn, k, 1);
        const Smem pwo = smem_layout(c->m, c->n, XWp, c->NWn, k, 0);
        if (pw.a_end <= budget) { g.pad = 1; g.XW = XWp; g.a_in_smem = 1; g.smem_eval = (size_t)pw.a_end; }
        else if (pwo.a_end <= budget) { g.pad = 1; g.XW = XWp; g.a_in_smem = 0; g.smem_eval = (size_t)pwo.a_end; }
        if (g.pad) return LNS_OK;
    }
    if (c->m > PACKED_MAX_M && !c->no_pad) {
        // segment-loop path: padded placement within the largest X (XW words, W < XW <= 2W + 1)
        // that fits next to the plan (A from global memory)
        for (int XWp = 2 * c->W + 1; XWp > c->W; XWp--) {
            const Smem pwo = smem_layout(c->m, c->n, XWp, c->NWn, k, 0, 0, g.pkw);
            if (pwo.a_end <= budget) { g.pad = 1; g.XW = XWp; g.a_in_smem = 0; g.smem_eval = (size_t)pwo.a_end; break; }
        }
        if (g.pad) return LNS_OK;
    }
    const Smem with = smem_layout(c->m, c->n, c->W, c->NWn, k, 1, 0, g.pkw);
    const Smem without = smem_layout(c->m, c->n, c->W, c->NWn, k, 0, 0, g.pkw);
    const Smem xg = smem_layout(c->m, c->n, c->W, c->NWn, k, 0, 1, g.pkw);
    if (with.a_end <= budget) { g.a_in_smem = 1; g.smem_eval = (size_t)with.a_end; }
    else if (without.a_end <= budget) { g.a_in_smem = 0; g.smem_eval = (size_t)without.a_end; }
    else if (xg.a_end <= budget) { g.a_in_smem = 0; g.x_global = 1; g.smem_eval = (size_t)xg.a_end; }
    else return fail(LNS_ERANGE, "plan does not fit in shared memory (n or m too large)");
    return LNS_OK;
}

lns_status check_k(lns_ctx *c, int k, Geometry &g)
{
    if (!c) return fail(LNS_EINVAL, "null context");
    if (k < 1 || k > 3)
        return fail(LNS_EINVAL, k <= KG_MAX ? "k = 4..7: lns_tabu_run, lns_eval_all and lns_unrank only"
                                            : "k must be in 1..7");
    if (c->n < k) return fail(LNS_EINVAL, "n < k");
    const int64_t Mk = comb_k(c->n, k);
    if (Mk >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "C(n,k) >= 2^32-1");
    g.M = (uint32_t)Mk;
    // m > 255: the packed-record region first, unless it pushes X out of shared
    // memory where the segment plan alone would keep it there
    lns_status s = geometry(c, k, g, (c->m > PACKED_MAX_M && !c->no_pkw) ? 1 : 0);
    if (g.pkw && (s != LNS_OK || g.x_global)) {
        Geometry g0 = g;
        if (geometry(c, k, g0, 0) == LNS_OK && (s != LNS_OK || !g0.x_global)) { g = g0; s = LNS_OK; }
    }
    if (s != LNS_OK) return s;
    g.pkw_force = c->force_pkw;
    if (g.x_global) {  // one X slot per CTA of the largest grid any launch uses (eval_all: 8 x SMs)
        s = grow(c->d_X, c->X_cap, (size_t)8 * c->numSMs * c->W * c->n);
        if (s != LNS_OK) return s;
    }
    return LNS_OK;
}

// CTAs for one search over `span` ranks: about one CTA per 2,048 neighbour x (row words + 2) of
// evaluation work (per-neighbour cost grows with the row words), capped by the SMs.
int search_blocks(const lns_ctx *c, uint32_t span, int occ)
{
    const int cap = std::min(c->numSMs * occ, MAX_SLOTS);
    if (c->blocks_override > 0) return std::min(c->blocks_override, cap);
    const int64_t work = (int64_t)span * (c->W + 2);
    const int nb = (int)std::min<int64_t>((int64_t)cap, std::max<int64_t>(1, (work + 2047) / 2048));
    return std::max(1, nb);
}

SearchArgs make_args(lns_ctx *c, const Geometry &g, int64_t iters, int64_t L, int flags)
{
    SearchArgs A;
    A.I = dev_inst(c);
    A.I.XW = g.XW > 0 ? g.XW : c->W;
    A.I.pkw = g.pkw;
    A.I.pad = 0;  // per launch: pad_for()
    A.M = g.M;
    slice_of(g.M, c->part, c->nparts, A.lo, A.hi);
    A.iters = iters; A.L = L; A.stop_on_zero = (flags & LNS_STOP_ON_ZERO) ? 1 : 0;
    A.aspiration = (flags & LNS_ASPIRATION) ? 1 : 0;
    A.sol_list = (flags & LNS_TABU_SOLUTIONS) ? 1 : 0;
    A.ring = c->d_ring;
    A.Xg = g.x_global ? c->d_X : nullptr;
    A.a_in_smem = g.a_in_smem;
    A.until_smem = 0; A.tri_smem = 0; A.slice_cap = 0;
    A.groups = 1; A.R = 0; A.V0s = nullptr; A.res = nullptr; A.vouts = nullptr;
    A.nph = 0;
    A.vb = c->d_vb; A.Y = c->d_Y; A.fs = c->d_fs; A.until = c->d_until;
    A.slots = c->d_slots; A.counter = c->d_counter; A.trace_r = c->d_tr; A.trace_f = c->d_tf;
    A.tbits = c->d_tbits; A.tring = c->d_tring; A.bits_mode = 0; A.ring_on = 0;
    A.bit_words = (uint32_t)(((uint64_t)g.M + 31) / 32);
    A.peers = nullptr; A.npeers = 0; A.part = 0; A.nb_total = 0; A.timeout_ns = 0;
    A.grid_timeout_ns = c->grid_timeout_ms * 1000000LL;
    A.plain_launch = (flags & LNS_PLAIN_LAUNCH) ? 1 : 0;
    A.enc_keys = 0;
    return A;
}

// Prepare a search: V0 -> state, until[] cleared, trace buffers sized.
lns_status search_setup(lns_ctx *c, const Geometry &g, int64_t iters, uint64_t seed, const int8_t *V0, cudaStream_t st,
                        bool need_until = true)
{
    lns_status s;
    std::vector<int8_t> hv;
    if (V0) CK(cudaMemcpyAsync(c->d_V, V0, c->n, cudaMemcpyDefault, st));
    else {
        hv.resize(c->n);
        vector_from_seed(c->n, seed, hv.data());
        CK(cudaMemcpyAsync(c->d_V, hv.data(), c->n, cudaMemcpyHostToDevice, st));
    }
    if (need_until) {  // the global until[] (stepped path, variants); persistent searches keep their own state
        if ((s = grow(c->d_until, c->until_cap, g.M)) != LNS_OK) return s;
        CK(cudaMemsetAsync(c->d_until, 0, (size_t)g.M * 4, st));
    }
    const size_t tc = (size_t)std::max<int64_t>(iters, 1);
    if ((s = grow(c->d_tr, c->trace_cap, tc)) != LNS_OK) return s;
    if ((s = grow(c->d_tf, c->trace_cap_f, tc)) != LNS_OK) return s;
    k_fill_i64<<<1, 32, 0, st>>>(c->d_slots + SLOT_ACC, KEY_NONE, 2);
    CK(cudaMemsetAsync(c->d_counter, 0, sizeof(unsigned), st));
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, nullptr, c->d_fs);
    CK(cudaGetLastError());
    return LNS_OK;
}

lns_status search_finish(lns_ctx *c, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit, lns_result *res,
                         cudaStream_t st)
{
    int64_t fs[FS_N];
    CK(cudaMemcpyAsync(fs, c->d_fs, sizeof(fs), cudaMemcpyDeviceToHost, st));
    std::vector<uint32_t> vb(c->NWn);
    CK(cudaMemcpyAsync(vb.data(), c->d_vb, 4 * c->NWn, cudaMemcpyDeviceToHost, st));
    CK(cudaStreamSynchronize(st));
    if (fs[FS_ERR] == 1) return fail(LNS_EINVAL, "V0 entries must be +1 or -1");
    if (fs[FS_ERR] == 2) return fail(LNS_ENOADMISSIBLE, "no admissible move");
    if (fs[FS_ERR] == 3) return fail(LNS_EPEER, "a partition did not reach the exchange in time");
    if (fs[FS_ERR] == 4) return fail(LNS_EPEER, "a CTA of the grid did not reach the exchange in time (not co-resident?)");
    const int64_t done = fs[FS_T];
    if (trace_rank && done > 0) CK(cudaMemcpyAsync(trace_rank, c->d_tr, done * 8, cudaMemcpyDefault, st));
    if (trace_fit && done > 0) CK(cudaMemcpyAsync(trace_fit, c->d_tf, done * 8, cudaMemcpyDefault, st));
    std::vector<int8_t> hv;
    if (V_out) {
        hv.resize(c->n);
        for (int i = 0; i < c->n; i++) hv[i] = ((vb[i / 32] >> (i % 32)) & 1) ? -1 : 1;
        CK(cudaMemcpyAsync(V_out, hv.data(), c->n, cudaMemcpyDefault, st));
    }
    CK(cudaStreamSynchronize(st));
    if (res) {
        res->iters_done = done; res->final_f = fs[FS_F]; res->best_f = fs[FS_BEST];
        res->best_iter = fs[FS_BESTIT]; res->first_zero_iter = fs[FS_ZERO];
        res->solved = fs[FS_BEST] == 0; res->reserved = 0;
    }
    return LNS_OK;
}

// Shared-memory caches of a search with nb CTAs over [A.lo, A.hi): the until[] slice and the
// flip-set table when they fit next to the plan. Returns the dynamic shared-memory bytes.
size_t cache_geometry(SearchArgs &A, const Geometry &g, int nb, int budget)
{
    const uint64_t slice = ((((uint64_t)(A.hi - A.lo) + nb - 1) / nb + 64) + 3) & ~3ull;  // 16-B aligned caches
    size_t smem = g.smem_eval;
    A.slice_cap = (int32_t)std::min<uint64_t>(slice, 1u << 30);
    A.until_smem = 0; A.tri_smem = 0;
    if (A.sol_list) {  // until[] stays in global memory: every CTA of the group writes into it
        if (g.smem_eval + 12 * slice <= (size_t)budget) { A.tri_smem = 1; smem = g.smem_eval + 12 * slice; }
        return smem;
    }
    if (g.smem_eval + 12 * slice <= (size_t)budget) {  // until[] slice + flip-set table
        A.until_smem = 1; A.tri_smem = 1;
        smem = g.smem_eval + 12 * slice;
    } else if (g.smem_eval + 4 * slice <= (size_t)budget) {
        A.until_smem = 1;
        smem = g.smem_eval + 4 * slice;
    }
    return smem;
}

// Raise a kernel's dynamic shared-memory limit once per (kernel, device): cudaFuncSetAttribute on a
// kernel that is running (another context's search on another stream) waits for it, which would
// serialise concurrent searches of one process.
cudaError_t allow_smem(const void *fn, int bytes)
{
    static std::mutex mu;
    static std::map<std::pair<const void *, int>, int> done;
    int dev = 0;
    cudaGetDevice(&dev);
    std::lock_guard<std::mutex> lk(mu);
    int &have = done[{fn, dev}];
    if (have >= bytes) return cudaSuccess;
    const cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes);
    if (e == cudaSuccess) have = bytes;
    return e;
}

// Padded placement pays off when a CTA evaluates many neighbours per plan (it adds a serial warp
// pass to every plan build): the same slice test as the contiguous-run evaluation path.
// m > 255: the packed plan (§5.11) pays off when a CTA evaluates many neighbours per plan (its
// build adds a barrier and a serial placement); otherwise the segment plan is used throughout.
inline int pkw_for(const Geometry &g, uint32_t span, int nb)
{
    return (g.pkw && (g.pkw_force || span / (uint32_t)std::max(nb, 1) >= 2u * NT)) ? 1 : 0;
}

inline int pad_for(const Geometry &g, uint32_t span, int nb)
{
    return (g.pad && span / (uint32_t)std::max(nb, 1) >= 4u * NT) ? 1 : 0;
}

// bits_mode: when the until[] slice of a CTA does not fit in shared memory and the
// default tabu list is used (no aspiration, no solution list), keep one bit per rank plus a ring of
// the last L accepted ranks instead of a u32 per rank: ceil(M/32) words per group (C5: 22 MB instead
// of 713 MB), and the ring only when a search can outlast its tenure (L < iterations). groups
// bitmaps and rings are allocated; zero_now clears the bitmaps on `st` (a single search: batched
// restarts clear their words in the kernel).
lns_status setup_bits(lns_ctx *c, SearchArgs &A, int groups, bool zero_now, cudaStream_t st)
{
    A.bits_mode = 0; A.ring_on = 0;
    if (c->no_bits || A.until_smem || A.sol_list || A.aspiration) return LNS_OK;
    lns_status s;
    const size_t per = A.bit_words;
    if ((s = grow(c->d_tbits, c->tbits_cap, per * (size_t)groups)) != LNS_OK) return s;
    A.tbits = c->d_tbits;
    if (zero_now) CK(cudaMemsetAsync(c->d_tbits, 0, per * groups * 4, st));
    if (A.L > 0 && A.L < A.iters) {
        if ((s = grow(c->d_tring, c->tring_cap, (size_t)A.L * groups)) != LNS_OK) return s;
        A.tring = c->d_tring;
        A.ring_on = 1;
    }
    A.bits_mode = 1;
    return LNS_OK;
}

template <int K>
lns_status launch_search(lns_ctx *c, SearchArgs A, const Geometry &g, cudaStream_t st, int nb_force = 0)
{
    const void *kern = (const void *)k_search<K, false>;
    // persistent geometry: first the CTA count at the eval footprint, then cache the until[]
    // slice in shared memory if it fits next to it
    const int budget = c->smemOptin - 1024;  // static shared memory of the kernels stays < 1 KiB
    CK(allow_smem(kern, budget));
    int occ = 0;
    CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k_search<K, false>, NT, g.smem_eval));
    if (occ < 1) return fail(LNS_ERANGE, "persistent kernel does not fit on an SM");
    const int nb = nb_force > 0 ? nb_force : search_blocks(c, A.hi - A.lo, 1);
    if (A.npeers > 0) A.nb_total = (int64_t)nb * A.npeers;
    // one search over all its CTAs (latency-bound): keys carry the flip set, so the winner needs no
    // unranking after the exchange (every partition of a peer run takes the same choice: same n, k)
    // (not when a CTA's slice takes eval_range's contiguous-run path: its keys carry ranks)
    A.enc_keys = ((K == 3 && A.I.n <= 1024) || (K == 2 && A.I.n <= 65536)) &&
                 (A.hi - A.lo) / (uint32_t)nb + 64u < 4u * NT ? 1 : 0;
    A.I.pad = pad_for(g, A.hi - A.lo, nb);
    A.I.pkw = pkw_for(g, A.hi - A.lo, nb);
    const size_t smem = cache_geometry(A, g, nb, budget);
    lns_status sb = setup_bits(c, A, 1, true, st);
    if (sb != LNS_OK) return sb;
    if (!A.until_smem && !A.bits_mode && !c->d_until) return fail(LNS_EINVAL, "internal: no tabu state allocated");
    // exchange slots (3 keys on separate lines) = KEY_NONE, arrival counter = 0
    k_init_slots<<<1, 64, 0, st>>>(c->d_slots, 1);
    void *args[] = {&A};
    CK(cudaEventRecord(c->ev0, st));
    if (A.plain_launch) CK(cudaLaunchKernel(kern, dim3(nb), dim3(NT), args, smem, st));
    else CK(cudaLaunchCooperativeKernel(kern, dim3(nb), dim3(NT), args, smem, st));
    CK(cudaEventRecord(c->ev1, st));
    return LNS_OK;
}

// Batched restarts: the phases of A (cooperative grid = the SMs); A carries V0s / res / vouts.
template <int K>
lns_status launch_batch(lns_ctx *c, SearchArgs A, const Geometry &g, int grid, int ngroups, int nb_min,
                        int64_t *gslots, cudaStream_t st)
{
    const int budget = c->smemOptin - 1024;
    CK(allow_smem((const void *)k_search<K, true>, budget));
    A.I.pad = pad_for(g, A.hi - A.lo, nb_min);
    A.I.pkw = pkw_for(g, A.hi - A.lo, nb_min);
    const size_t smem = cache_geometry(A, g, nb_min, budget);
    lns_status sb = setup_bits(c, A, ngroups, false, st);  // each restart clears its words in the kernel
    if (sb != LNS_OK) return sb;
    if (!A.until_smem && !A.bits_mode) {  // one global until[] per group of every phase
        lns_status s = grow(c->d_until, c->until_cap, (size_t)ngroups * g.M);
        if (s != LNS_OK) return s;
        A.until = c->d_until;
    }
    k_init_slots<<<(64 * ngroups + 255) / 256, 256, 0, st>>>(gslots, ngroups);
    A.slots = gslots;
    A.groups = 0;
    void *args[] = {&A};
    CK(cudaEventRecord(c->ev0, st));
    CK(cudaLaunchCooperativeKernel((void *)k_search<K, true>, dim3(grid), dim3(NT), args, smem, st));
    CK(cudaEventRecord(c->ev1, st));
    return LNS_OK;
}

template <int K>
lns_status launch_step_eval(lns_ctx *c, const SearchArgs &A, const Geometry &g, int64_t *key_out, int32_t *fit_out,
                            bool all, cudaStream_t st)
{
    const int budget = c->smemOptin - 1024;
    CK(allow_smem((const void *)k_step_eval<K, false>, budget));
    CK(allow_smem((const void *)k_step_eval<K, true>, budget));
    int occ = 0;
    CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k_step_eval<K, false>, NT, g.smem_eval));
    if (occ < 1) return fail(LNS_ERANGE, "eval kernel does not fit on an SM");
    SearchArgs a = A;
    a.slots = c->d_slots + SLOT_ACC;
    int nb = search_blocks(c, A.hi - A.lo, occ);
    if (all) {
        nb = (int)std::min<int64_t>(std::max<int64_t>(1, (A.hi - A.lo) / 1024), 4LL * c->numSMs * occ);
        if (c->blocks_override > 0) nb = std::min(c->blocks_override, 4 * c->numSMs * occ);
        a.I.pad = pad_for(g, A.hi - A.lo, nb);
        a.I.pkw = pkw_for(g, A.hi - A.lo, nb);
        k_step_eval<K, true><<<nb, NT, g.smem_eval, st>>>(a, key_out, fit_out);
    } else {
        a.I.pad = pad_for(g, A.hi - A.lo, nb);
        a.I.pkw = pkw_for(g, A.hi - A.lo, nb);
        k_step_eval<K, false><<<nb, NT, g.smem_eval, st>>>(a, key_out, fit_out);
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

lns_status dispatch_search(lns_ctx *c, int k, const SearchArgs &A, const Geometry &g, cudaStream_t st, int nb_force = 0)
{
    switch (k) {
    case 1: return launch_search<1>(c, A, g, st, nb_force);
    case 2: return launch_search<2>(c, A, g, st, nb_force);
    default: return launch_search<3>(c, A, g, st, nb_force);
    }
}
lns_status dispatch_step_eval(lns_ctx *c, int k, const SearchArgs &A, const Geometry &g, int64_t *key_out,
                              int32_t *fit_out, bool all, cudaStream_t st)
{
    switch (k) {
    case 1: return launch_step_eval<1>(c, A, g, key_out, fit_out, all, st);
    case 2: return launch_step_eval<2>(c, A, g, key_out, fit_out, all, st);
    default: return launch_step_eval<3>(c, A, g, key_out, fit_out, all, st);
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

// k = 4..7 (the generic-k kernel k_gen): the instantiation, limits and shared memory.
const void *kgen_fn(int k)
{
    switch (k) {
    case 4: return (const void *)k_gen<4>;
    case 5: return (const void *)k_gen<5>;
    case 6: return (const void *)k_gen<6>;
    default: return (const void *)k_gen<7>;
    }
}

cudaError_t kgen_launch(int k, int nb, size_t smem, cudaStream_t st, const GenArgs &A)
{
    switch (k) {
    case 4: k_gen<4><<<nb, NTG, smem, st>>>(A); break;
    case 5: k_gen<5><<<nb, NTG, smem, st>>>(A); break;
    case 6: k_gen<6><<<nb, NTG, smem, st>>>(A); break;
    default: k_gen<7><<<nb, NTG, smem, st>>>(A); break;
    }
    return cudaGetLastError();
}

// k = 4..7: limits and shared memory.
lns_status gen_check(lns_ctx *c, int k, uint32_t &M, size_t &smem)
{
    if (!c) return fail(LNS_EINVAL, "null context");
    if (k < 4 || k > KG_MAX) return fail(LNS_EINVAL, "k must be in 1..7");
    if (c->n < k) return fail(LNS_EINVAL, "n < k");
    if (c->m > PACKED_MAX_M) return fail(LNS_ERANGE, "k > 3 needs m <= 255 (byte window)");
    const int64_t Mk = comb_k(c->n, k);
    if (Mk < 0 || Mk >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "C(n,k) >= 2^32-1");
    M = (uint32_t)Mk;
    smem = (size_t)gen_layout(c->m, c->n, c->NWn, k).end;
    if (smem > (size_t)(c->smemOptin - 1024)) return fail(LNS_ERANGE, "k > 3 plan does not fit in shared memory");
    return LNS_OK;
}

GenArgs gen_args(lns_ctx *c, int k, uint32_t M, int64_t iters, int64_t L, int flags)
{
    GenArgs A;
    A.I = dev_inst(c);
    A.K = k; A.M = M; A.iters = iters; A.L = L;
    A.stop_on_zero = (flags & LNS_STOP_ON_ZERO) ? 1 : 0;
    A.aspiration = (flags & LNS_ASPIRATION) ? 1 : 0;
    A.vb = c->d_vb; A.Y = c->d_Y; A.fs = c->d_fs; A.until = c->d_until; A.slots = c->d_slots;
    A.trace_r = c->d_tr; A.trace_f = c->d_tf; A.fit_out = nullptr; A.best_out = nullptr;
    A.R = 0; A.G = 1; A.nbg = 1; A.V0s = nullptr; A.res = nullptr; A.vouts = nullptr;
    A.grid_timeout_ns = c->grid_timeout_ms * 1000000LL;
    return A;
}

lns_status resolve_tenure(int64_t M, int64_t tenure, int64_t &L);

// lns_tabu_run for k = 4..7: one persistent cooperative k_gen launch (single search, one device).
lns_status gen_tabu_run(lns_ctx *c, int32_t k, int64_t iters, int64_t tenure, uint64_t seed, const int8_t *V0,
                        int32_t flags, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit, lns_result *res,
                        void *stream)
{
    uint32_t M;
    size_t smem;
    lns_status s = gen_check(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (!res) return fail(LNS_EINVAL, "res is required");
    if (iters < 0 || iters >= (int64_t)INT32_MAX) return fail(LNS_EINVAL, "iters must be in [0, 2^31)");
    if ((flags & (LNS_FORCE_STEPPED | LNS_TABU_SOLUTIONS)) || c->comm || c->nparts > 1 || c->npeers > 0)
        return fail(LNS_EINVAL, "k > 3: one device, persistent kernel, rank tabu list (optionally aspiration) only");
    int64_t L;
    if ((s = resolve_tenure(M, tenure, L)) != LNS_OK) return s;
    if (iters + L >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "iters + tenure >= 2^32");
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    Geometry g;
    g.M = M;
    if ((s = search_setup(c, g, iters, seed, V0, st)) != LNS_OK) return s;
    if (iters > 0) {
        CK(allow_smem(kgen_fn(k), (int)smem));
        int occ = 0;
        CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kgen_fn(k), NTG, smem));
        if (occ < 1) return fail(LNS_ERANGE, "k > 3 kernel does not fit on an SM");
        int nb = (int)std::min<int64_t>(std::min(c->numSMs * occ, MAX_SLOTS), std::max<int64_t>(1, (int64_t)M / (4 * NTG)));
        if (c->blocks_override > 0) nb = std::min(c->blocks_override, c->numSMs * occ);
        k_init_slots<<<1, 64, 0, st>>>(c->d_slots, 1);
        GenArgs A = gen_args(c, k, M, iters, L, flags);
        void *args[] = {&A};
        CK(cudaEventRecord(c->ev0, st));
        CK(cudaLaunchCooperativeKernel((void *)kgen_fn(k), dim3(nb), dim3(NTG), args, smem, st));
        CK(cudaEventRecord(c->ev1, st));
    }
    s = search_finish(c, V_out, trace_rank, trace_fit, res, st);
    float ms = 0;
    if (iters > 0 && cudaEventElapsedTime(&ms, c->ev0, c->ev1) == cudaSuccess) c->last_ms = ms;
    cudaGetLastError();
    return s;
}

// lns_tabu_run_batch for k = 4..7: R restarts on G groups of nbg CTAs (one cooperative k_gen).
lns_status gen_tabu_run_batch(lns_ctx *c, int32_t k, int32_t R, int64_t iters, int64_t tenure, uint64_t seed,
                              const int8_t *V0, int32_t flags, int8_t *V_out, lns_result *res, void *stream)
{
    uint32_t M;
    size_t smem;
    lns_status s = gen_check(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (!res || R < 0) return fail(LNS_EINVAL, "bad argument");
    if (iters < 0 || iters >= (int64_t)INT32_MAX) return fail(LNS_EINVAL, "iters must be in [0, 2^31)");
    if (flags & (LNS_FORCE_STEPPED | LNS_TABU_SOLUTIONS))
        return fail(LNS_EINVAL, "k > 3: rank tabu list (optionally aspiration) only");
    int64_t L;
    if ((s = resolve_tenure(M, tenure, L)) != LNS_OK) return s;
    if (iters + L >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "iters + tenure >= 2^32");
    if (R == 0) return LNS_OK;
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    const int n = c->n, SMs = c->numSMs;
    std::vector<int8_t> hv((size_t)R * n);
    if (V0) {
        // ordered after the caller's work on `stream` (a device V0 may still be being written there)
        CK(cudaMemcpyAsync(hv.data(), V0, hv.size(), cudaMemcpyDefault, st));
        CK(cudaStreamSynchronize(st));
        for (int8_t v : hv)
            if (v != 1 && v != -1) return fail(LNS_EINVAL, "V0 entries must be +1 or -1");
    } else {
        for (int r = 0; r < R; r++) {
            uint64_t sr = seed + (uint64_t)r;
            vector_from_seed(n, splitmix64_next(sr), hv.data() + (size_t)r * n);
        }
    }
    CK(allow_smem(kgen_fn(k), (int)smem));
    int occ = 0;
    CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kgen_fn(k), NTG, smem));
    if (occ < 1) return fail(LNS_ERANGE, "k > 3 kernel does not fit on an SM");
    // groups: one round of R searches on S / R CTAs each when R <= S (S = SMs x resident CTAs),
    // else S single-CTA groups; an until[] of M entries per group (8 GiB at most)
    const int S = SMs * occ;
    int nbg = c->blocks_override > 0 ? std::min(c->blocks_override, S) : std::max(1, S / std::max(1, R));
    int G = std::min(R, std::max(1, S / nbg));
    G = (int)std::min<int64_t>(G, std::max<int64_t>(1, (8LL << 30) / (4LL * M)));
    if ((s = grow(c->d_V0s, c->v0s_cap, hv.size())) != LNS_OK) return s;
    if ((s = grow(c->d_res, c->res_cap, (size_t)R * FS_N)) != LNS_OK) return s;
    if ((s = grow(c->d_vouts, c->vouts_cap, (size_t)R * c->NWn)) != LNS_OK) return s;
    if ((s = grow(c->d_gslots, c->gslots_cap, (size_t)G * 64)) != LNS_OK) return s;
    if ((s = grow(c->d_until, c->until_cap, (size_t)G * M)) != LNS_OK) return s;
    CK(cudaMemcpyAsync(c->d_V0s, hv.data(), hv.size(), cudaMemcpyHostToDevice, st));
    k_init_slots<<<(64 * G + 255) / 256, 256, 0, st>>>(c->d_gslots, G);
    GenArgs A = gen_args(c, k, M, iters, L, flags);
    A.R = R; A.G = G; A.nbg = nbg; A.V0s = c->d_V0s; A.res = c->d_res; A.vouts = c->d_vouts;
    A.until = c->d_until; A.slots = c->d_gslots; A.trace_r = nullptr; A.trace_f = nullptr;
    void *args[] = {&A};
    CK(cudaEventRecord(c->ev0, st));
    CK(cudaLaunchCooperativeKernel((void *)kgen_fn(k), dim3(G * nbg), dim3(NTG), args, smem, st));
    CK(cudaEventRecord(c->ev1, st));
    std::vector<int64_t> hres((size_t)R * FS_N);
    std::vector<uint32_t> hvo((size_t)R * c->NWn);
    CK(cudaMemcpyAsync(hres.data(), c->d_res, hres.size() * 8, cudaMemcpyDeviceToHost, st));
    CK(cudaMemcpyAsync(hvo.data(), c->d_vouts, hvo.size() * 4, cudaMemcpyDeviceToHost, st));
    CK(cudaStreamSynchronize(st));
    float ms = 0;
    if (cudaEventElapsedTime(&ms, c->ev0, c->ev1) == cudaSuccess) c->last_ms = ms;
    for (int r = 0; r < R; r++) {
        const int64_t *o = hres.data() + (size_t)r * FS_N;
        if (o[FS_ERR] == 4) return fail(LNS_EPEER, "a CTA of the grid did not reach the exchange in time");
        if (o[FS_ERR] == 2) return fail(LNS_ENOADMISSIBLE, "no admissible move");
        res[r].iters_done = o[FS_T]; res[r].final_f = o[FS_F]; res[r].best_f = o[FS_BEST];
        res[r].best_iter = o[FS_BESTIT]; res[r].first_zero_iter = o[FS_ZERO];
        res[r].solved = o[FS_BEST] == 0; res[r].reserved = 0;
    }
    if (V_out) {
        std::vector<int8_t> ho((size_t)R * n);
        for (int r = 0; r < R; r++)
            for (int i = 0; i < n; i++)
                ho[(size_t)r * n + i] = ((hvo[(size_t)r * c->NWn + i / 32] >> (i % 32)) & 1) ? -1 : 1;
        CK(cudaMemcpyAsync(V_out, ho.data(), ho.size(), cudaMemcpyDefault, st));
        CK(cudaStreamSynchronize(st));
    }
    return LNS_OK;
}

// lns_eval_neighborhood for k = 4..7: k_gen over every rank, admissible keys MIN-reduced.
lns_status gen_eval_best(lns_ctx *c, int32_t k, const int8_t *V, const int32_t *Y, const uint32_t *tabu_bits,
                         int64_t *best_fitness, int64_t *best_rank, void *stream)
{
    uint32_t M;
    size_t smem;
    lns_status s = gen_check(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (!V || !Y || !best_fitness || !best_rank) return fail(LNS_EINVAL, "null argument");
    if (c->nparts > 1 || c->comm || c->npeers > 0) return fail(LNS_EINVAL, "k > 3: no partitions");
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    const size_t tw = (M + 31) / 32;
    if ((s = grow(c->d_until, c->until_cap, M)) != LNS_OK) return s;
    if (tabu_bits) {
        if ((s = grow(c->d_bits, c->bits_cap, tw)) != LNS_OK) return s;
        CK(cudaMemcpyAsync(c->d_bits, tabu_bits, tw * 4, cudaMemcpyDefault, st));
    }
    k_bits_to_until<<<std::min<uint32_t>(4096, (M + 255) / 256), 256, 0, st>>>(tabu_bits ? c->d_bits : nullptr,
                                                                              c->d_until, M);
    CK(cudaMemcpyAsync(c->d_V, V, c->n, cudaMemcpyDefault, st));
    CK(cudaMemcpyAsync(c->d_Yin, Y, 4 * (size_t)c->m, cudaMemcpyDefault, st));
    k_fill_i64<<<1, 32, 0, st>>>(c->d_slots + SLOT_OUT, KEY_NONE, 1);
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, c->d_Yin, c->d_fs);
    CK(allow_smem(kgen_fn(k), (int)smem));
    GenArgs A = gen_args(c, k, M, 0, 0, 0);
    A.best_out = (unsigned long long *)(c->d_slots + SLOT_OUT);
    int nb = (int)std::min<int64_t>(4LL * c->numSMs, std::max<int64_t>(1, (int64_t)M / (4 * NTG)));
    if (c->blocks_override > 0) nb = std::min(c->blocks_override, 4 * c->numSMs);
    CK(cudaEventRecord(c->ev0, st));
    CK(kgen_launch(k, nb, smem, st, A));
    CK(cudaEventRecord(c->ev1, st));
    int64_t key, fs[FS_N];
    CK(cudaMemcpyAsync(&key, c->d_slots + SLOT_OUT, 8, cudaMemcpyDeviceToHost, st));
    CK(cudaMemcpyAsync(fs, c->d_fs, sizeof(fs), cudaMemcpyDeviceToHost, st));
    CK(cudaStreamSynchronize(st));
    float ms = 0; cudaEventElapsedTime(&ms, c->ev0, c->ev1); c->last_ms = ms;
    if (fs[FS_ERR]) return fail(LNS_EINVAL, "V must be +-1 and Y must equal A V");
    if (key == KEY_NONE) { *best_fitness = -1; *best_rank = -1; return fail(LNS_ENOADMISSIBLE, "all ranks tabu"); }
    *best_fitness = key >> 32;
    *best_rank = key & 0xffffffffLL;
    return LNS_OK;
}

// lns_eval_all for k = 4..7.
lns_status gen_eval_all(lns_ctx *c, int32_t k, const int8_t *V, int32_t *fitness_out, void *stream)
{
    uint32_t M;
    size_t smem;
    lns_status s = gen_check(c, k, M, smem);
    if (s != LNS_OK) return s;
    if (!V || !fitness_out) return fail(LNS_EINVAL, "null argument");
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    if ((s = grow(c->d_fit, c->fit_cap, M)) != LNS_OK) return s;
    CK(cudaMemcpyAsync(c->d_V, V, c->n, cudaMemcpyDefault, st));
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, nullptr, c->d_fs);
    CK(allow_smem(kgen_fn(k), (int)smem));
    GenArgs A = gen_args(c, k, M, 0, 0, 0);
    A.fit_out = c->d_fit;
    int nb = (int)std::min<int64_t>(4LL * c->numSMs, std::max<int64_t>(1, (int64_t)M / (4 * NTG)));
    if (c->blocks_override > 0) nb = std::min(c->blocks_override, 4 * c->numSMs);
    CK(cudaEventRecord(c->ev0, st));
    CK(kgen_launch(k, nb, smem, st, A));
    CK(cudaEventRecord(c->ev1, st));
    int64_t fs[FS_N];
    CK(cudaMemcpyAsync(fs, c->d_fs, sizeof(fs), cudaMemcpyDeviceToHost, st));
    CK(cudaMemcpyAsync(fitness_out, c->d_fit, 4 * (size_t)M, cudaMemcpyDefault, st));
    CK(cudaStreamSynchronize(st));
    float ms = 0; cudaEventElapsedTime(&ms, c->ev0, c->ev1); c->last_ms = ms;
    if (fs[FS_ERR]) return fail(LNS_EINVAL, "V must be +-1");
    return LNS_OK;
}

// NCCL entry points (resolved at run time: the library does not link NCCL)
struct NcclUid { uint8_t b[LNS_UNIQUE_ID_BYTES]; };  // ncclUniqueId, passed by value to ncclCommInitRank
typedef int (*nccl_get_uid_fn)(NcclUid *);
typedef int (*nccl_init_rank_fn)(void **, int, NcclUid, int);
typedef int (*nccl_destroy_fn)(void *);

// The libnccl to use: the copy already loaded in the process (by soname, or its symbols in the
// global scope); with allow_load, else a fresh dlopen (only for communicators this library
// creates itself, so every call on them goes to that same copy).
void *nccl_handle(bool allow_load)
{
    void *h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_NOLOAD);
    if (h) return h;
    if (dlsym(RTLD_DEFAULT, "ncclAllReduce")) return RTLD_DEFAULT;
    if (!allow_load) return nullptr;
    h = dlopen("libnccl.so.2", RTLD_NOW);
    if (!h) h = dlopen("libnccl.so", RTLD_NOW);
    return h;
}

void drop_owned_comm(lns_ctx *c)
{
    if (c->comm_owned && c->nccl_lib) {
        nccl_destroy_fn d = (nccl_destroy_fn)dlsym(c->nccl_lib, "ncclCommDestroy");
        if (d) d(c->comm_owned);
    }
    if (c->comm_owned && c->comm == c->comm_owned) { c->comm = nullptr; c->part = 0; c->nparts = 1; }
    c->comm_owned = nullptr;
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
    case LNS_EPEER: return "peer exchange timed out";
    default: return "unknown status";
    }
}

const char *lns_last_error(void) { return g_err.c_str(); }
int32_t lns_version(void) { return LNS_VERSION_NUM; }

void lns_pool_trim(void)
{
    Pool &P = pool();
    std::multimap<std::pair<int, size_t>, void *> drop;
    {
        std::lock_guard<std::mutex> lk(P.mu);
        drop.swap(P.cache);
        P.cached = 0;
    }
    int cur = 0;
    cudaGetDevice(&cur);
    for (auto &kv : drop) {
        cudaSetDevice(kv.first.first);
        cudaFree(kv.second);
    }
    cudaSetDevice(cur);
}

void lns_pool_stats(int64_t *cached_bytes, int64_t *live_bytes)
{
    Pool &P = pool();
    std::lock_guard<std::mutex> lk(P.mu);
    if (cached_bytes) *cached_bytes = (int64_t)P.cached;
    if (live_bytes) *live_bytes = (int64_t)P.live_bytes;
}

int64_t lns_neighborhood_size(int32_t n, int32_t k)
{
    if (k < 1 || k > KG_MAX) return -1;
    return n < k ? 0 : comb_k(n, k);
}

lns_status lns_create(const int8_t *A, int32_t m, int32_t n, const int32_t *S, int32_t device, lns_ctx **out)
{
    if (!out || !A || !S) return fail(LNS_EINVAL, "null argument");
    *out = nullptr;
    if (m < 1 || n < 1) return fail(LNS_EINVAL, "m and n must be >= 1");
    if (m > 65535) return fail(LNS_ERANGE, "m > 65535");
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
            const int8_t a = hA[(size_t)j * n + i];
            if (a != 1 && a != -1) return fail(LNS_EINVAL, "A entries must be +1 or -1");
            if (a < 0) arow[(size_t)j * NWn + i / 32] |= 1u << (i % 32);
        }
        if (hS[j] < 0 || hS[j] > n) return fail(LNS_EINVAL, "S entries must lie in [0, n]");
        H[hS[j]]++;
    }
    lns_ctx *c = new lns_ctx();
    c->device = device; c->m = m; c->n = n; c->W = W; c->NWn = NWn;
    { const char *e = getenv("LNS_NO_PAD"); c->no_pad = (e && e[0] == '1') ? 1 : 0; }
    { const char *e = getenv("LNS_NO_PKW"); c->no_pkw = (e && e[0] == '1') ? 1 : 0; }
    { const char *e = getenv("LNS_FORCE_PKW"); c->force_pkw = (e && e[0] == '1') ? 1 : 0; }
    { const char *e = getenv("LNS_NO_GRAPH"); c->no_graph = (e && e[0] == '1') ? 1 : 0; }
    { const char *e = getenv("LNS_NO_BITS"); c->no_bits = (e && e[0] == '1') ? 1 : 0; }
    { const char *e = getenv("LNS_GRID_TIMEOUT_MS"); if (e && atoll(e) > 0) c->grid_timeout_ms = atoll(e); }
    for (int b = 0; b <= n; b++)
        if (H[b] > 0) c->maxS = b;
    auto cleanup = [&](lns_status s) { lns_destroy(c); return s; };
    if (cudaDeviceGetAttribute(&c->numSMs, cudaDevAttrMultiProcessorCount, device) != cudaSuccess ||
        cudaDeviceGetAttribute(&c->smemOptin, cudaDevAttrMaxSharedMemoryPerBlockOptin, device) != cudaSuccess)
        return cleanup(fail(LNS_ECUDA, "device attributes"));
    if (pool_alloc(&c->d_Arow, arow.size() * 4) != cudaSuccess || pool_alloc(&c->d_H, (n + 1) * 4) != cudaSuccess ||
        pool_alloc(&c->d_vb, NWn * 4) != cudaSuccess || pool_alloc(&c->d_Y, m * 4) != cudaSuccess ||
        pool_alloc(&c->d_fs, FS_N * 8) != cudaSuccess || pool_alloc(&c->d_slots, SLOT_N * 8) != cudaSuccess ||
        pool_alloc(&c->d_counter, sizeof(unsigned)) != cudaSuccess || pool_alloc(&c->d_V, n) != cudaSuccess ||
        pool_alloc(&c->d_Yin, m * 4) != cudaSuccess) {
        return cleanup(fail(LNS_ENOMEM, "cudaMalloc failed"));
    }
    if (cudaMemcpy(c->d_Arow, arow.data(), arow.size() * 4, cudaMemcpyHostToDevice) != cudaSuccess ||
        cudaMemcpy(c->d_H, H.data(), (n + 1) * 4, cudaMemcpyHostToDevice) != cudaSuccess ||
        cudaMemset(c->d_counter, 0, sizeof(unsigned)) != cudaSuccess ||
        cudaEventCreate(&c->ev0) != cudaSuccess || cudaEventCreate(&c->ev1) != cudaSuccess ||
        cudaEventCreate(&c->ev2) != cudaSuccess || cudaEventCreate(&c->ev3) != cudaSuccess)
        return cleanup(fail(LNS_ECUDA, "upload"));
    *out = c;
    return LNS_OK;
}

void lns_destroy(lns_ctx *c)
{
    if (!c) return;
    DeviceGuard g(c->device);
    if (c->step_active) cudaDeviceSynchronize();  // an open stepped search may still run kernels
    for (void *p : {(void *)c->d_Arow, (void *)c->d_H, (void *)c->d_vb, (void *)c->d_Y, (void *)c->d_fs,
                    (void *)c->d_slots, (void *)c->d_counter, (void *)c->d_V, (void *)c->d_Yin, (void *)c->d_bits,
                    (void *)c->d_until, (void *)c->d_tr, (void *)c->d_tf, (void *)c->d_fit, (void *)c->d_V0s,
                    (void *)c->d_res, (void *)c->d_vouts, (void *)c->d_gslots, (void *)c->d_X, (void *)c->d_ring,
                    (void *)c->d_tbits, (void *)c->d_tring})
        pool_free(p);
    for (void *p : c->ipc_opened) cudaIpcCloseMemHandle(p);
    drop_owned_comm(c);
    cudaFree(c->d_xbuf); cudaFree(c->d_peers);
    if (c->ev0) cudaEventDestroy(c->ev0);
    if (c->ev1) cudaEventDestroy(c->ev1);
    if (c->ev2) cudaEventDestroy(c->ev2);
    if (c->ev3) cudaEventDestroy(c->ev3);
    if (c->cap_stream) cudaStreamDestroy(c->cap_stream);
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
    c->part = part; c->nparts = nparts; c->npeers = 0;
    return LNS_OK;
}

lns_status lns_attach_comm(lns_ctx *c, void *comm, int32_t rank, int32_t world)
{
    if (!c) return fail(LNS_EINVAL, "null context");
    if (!comm) { drop_owned_comm(c); c->comm = nullptr; c->part = 0; c->nparts = 1; return LNS_OK; }
    if (world < 1 || rank < 0 || rank >= world) return fail(LNS_EINVAL, "bad rank/world");
    // a BORROWED communicator belongs to the NCCL already in the process (e.g. torch's): its
    // ncclAllReduce is looked up there and never in a freshly loaded copy, which could be another
    // build than the one that created the communicator
    void *h = nccl_handle(false);
    void *sym = h ? dlsym(h, "ncclAllReduce") : nullptr;
    if (!sym) return fail(LNS_ENCCL, "ncclAllReduce not found: no libnccl loaded in this process (load torch's, or use lns_comm_init_rank)");
    drop_owned_comm(c);
    c->nccl_allreduce = (nccl_allreduce_fn)sym;
    c->nccl_lib = h;
    c->comm = comm;
    c->part = rank; c->nparts = world; c->npeers = 0;
    return LNS_OK;
}

lns_status lns_get_unique_id(uint8_t *id_out)
{
    if (!id_out) return fail(LNS_EINVAL, "null argument");
    void *h = nccl_handle(true);
    nccl_get_uid_fn fn = h ? (nccl_get_uid_fn)dlsym(h, "ncclGetUniqueId") : nullptr;
    if (!fn) return fail(LNS_ENCCL, "libnccl.so.2 not found");
    NcclUid uid;
    if (fn(&uid) != 0) return fail(LNS_ENCCL, "ncclGetUniqueId failed");
    memcpy(id_out, uid.b, LNS_UNIQUE_ID_BYTES);
    return LNS_OK;
}

lns_status lns_comm_init_rank(lns_ctx *c, const uint8_t *id, int32_t rank, int32_t world)
{
    if (!c || !id) return fail(LNS_EINVAL, "null argument");
    if (world < 1 || rank < 0 || rank >= world) return fail(LNS_EINVAL, "bad rank/world");
    void *h = nccl_handle(true);
    nccl_init_rank_fn init = h ? (nccl_init_rank_fn)dlsym(h, "ncclCommInitRank") : nullptr;
    void *ar = h ? dlsym(h, "ncclAllReduce") : nullptr;
    if (!init || !ar || !dlsym(h, "ncclCommDestroy")) return fail(LNS_ENCCL, "libnccl.so.2 not found");
    DeviceGuard dg(c->device);
    NcclUid uid;
    memcpy(uid.b, id, LNS_UNIQUE_ID_BYTES);
    void *comm = nullptr;
    if (init(&comm, world, uid, rank) != 0 || !comm) return fail(LNS_ENCCL, "ncclCommInitRank failed");
    drop_owned_comm(c);
    c->comm_owned = comm;
    c->comm = comm;
    c->nccl_allreduce = (nccl_allreduce_fn)ar;
    c->nccl_lib = h;
    c->part = rank; c->nparts = world; c->npeers = 0;
    return LNS_OK;
}

lns_status lns_exchange_buffer(lns_ctx *c, void **buf_dev)
{
    if (!c || !buf_dev) return fail(LNS_EINVAL, "null argument");
    DeviceGuard dg(c->device);
    if (!c->d_xbuf) {
        if (cudaMalloc(&c->d_xbuf, 64 * sizeof(unsigned long long)) != cudaSuccess) {
            cudaGetLastError();
            return fail(LNS_ENOMEM, "exchange buffer");
        }
        lns_status s = lns_exchange_reset(c, nullptr);
        if (s != LNS_OK) return s;
    }
    *buf_dev = c->d_xbuf;
    return LNS_OK;
}

lns_status lns_exchange_ipc_handle(lns_ctx *c, void *handle_out)
{
    if (!c || !handle_out) return fail(LNS_EINVAL, "null argument");
    static_assert(sizeof(cudaIpcMemHandle_t) == LNS_IPC_HANDLE_BYTES, "IPC handle size");
    void *buf = nullptr;
    lns_status s = lns_exchange_buffer(c, &buf);
    if (s != LNS_OK) return s;
    DeviceGuard dg(c->device);
    cudaIpcMemHandle_t h;
    CK(cudaIpcGetMemHandle(&h, buf));
    memcpy(handle_out, &h, sizeof(h));
    return LNS_OK;
}

lns_status lns_exchange_reset(lns_ctx *c, void *stream)
{
    if (!c || !c->d_xbuf) return fail(LNS_EINVAL, "no exchange buffer (lns_exchange_buffer first)");
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    k_init_slots<<<1, 64, 0, st>>>((int64_t *)c->d_xbuf, 1);
    CK(cudaGetLastError());
    CK(cudaStreamSynchronize(st));
    return LNS_OK;
}

lns_status lns_attach_peers(lns_ctx *c, int32_t part, int32_t nparts, void *const *bufs, int64_t timeout_ms)
{
    if (!c) return fail(LNS_EINVAL, "null context");
    DeviceGuard dg(c->device);
    if (nparts <= 1 || !bufs) { c->npeers = 0; c->part = 0; c->nparts = 1; return LNS_OK; }
    if (part < 0 || part >= nparts || nparts > MAX_PEERS) return fail(LNS_EINVAL, "bad partition (at most 16)");
    if (timeout_ms <= 0) return fail(LNS_EINVAL, "timeout_ms must be positive");
    void *own = nullptr;
    lns_status s = lns_exchange_buffer(c, &own);
    if (s != LNS_OK) return s;
    if (bufs[part] != own) return fail(LNS_EINVAL, "bufs[part] must be this context's exchange buffer");
    for (int q = 0; q < nparts; q++)
        if (!bufs[q]) return fail(LNS_EINVAL, "null peer buffer");
    if (!c->d_peers && cudaMalloc(&c->d_peers, MAX_PEERS * sizeof(void *)) != cudaSuccess) {
        cudaGetLastError();
        return fail(LNS_ENOMEM, "peer table");
    }
    CK(cudaMemcpy(c->d_peers, bufs, nparts * sizeof(void *), cudaMemcpyHostToDevice));
    c->npeers = nparts; c->part = part; c->nparts = nparts; c->comm = nullptr;
    c->peer_timeout_ms = timeout_ms;
    return LNS_OK;
}

lns_status lns_attach_peers_ipc(lns_ctx *c, int32_t part, int32_t nparts, const void *handles, int64_t timeout_ms)
{
    if (!c || !handles || nparts < 1 || part < 0 || part >= nparts || nparts > MAX_PEERS)
        return fail(LNS_EINVAL, "bad partition / handles");
    DeviceGuard dg(c->device);
    for (void *p : c->ipc_opened) cudaIpcCloseMemHandle(p);
    c->ipc_opened.clear();
    std::vector<void *> bufs(nparts, nullptr);
    lns_status s = lns_exchange_buffer(c, &bufs[part]);
    if (s != LNS_OK) return s;
    for (int q = 0; q < nparts; q++) {
        if (q == part) continue;
        cudaIpcMemHandle_t h;
        memcpy(&h, (const char *)handles + (size_t)q * LNS_IPC_HANDLE_BYTES, sizeof(h));
        void *p = nullptr;
        CK(cudaIpcOpenMemHandle(&p, h, cudaIpcMemLazyEnablePeerAccess));
        c->ipc_opened.push_back(p);
        bufs[q] = p;
    }
    return lns_attach_peers(c, part, nparts, bufs.data(), timeout_ms);
}

lns_status lns_eval_neighborhood(lns_ctx *c, int32_t k, const int8_t *V, const int32_t *Y, const uint32_t *tabu_bits,
                                 int64_t *best_fitness, int64_t *best_rank, void *stream)
{
    if (k >= 4) return gen_eval_best(c, k, V, Y, tabu_bits, best_fitness, best_rank, stream);
    Geometry g;
    lns_status s = check_k(c, k, g);
    if (s != LNS_OK) return s;
    if (!V || !Y || !best_fitness || !best_rank) return fail(LNS_EINVAL, "null argument");
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    const size_t tw = (g.M + 31) / 32;
    if ((s = grow(c->d_until, c->until_cap, g.M)) != LNS_OK) return s;
    if (tabu_bits) {
        if ((s = grow(c->d_bits, c->bits_cap, tw)) != LNS_OK) return s;
        CK(cudaMemcpyAsync(c->d_bits, tabu_bits, tw * 4, cudaMemcpyDefault, st));
    }
    k_bits_to_until<<<std::min<uint32_t>(4096, (g.M + 255) / 256), 256, 0, st>>>(tabu_bits ? c->d_bits : nullptr,
                                                                                c->d_until, g.M);
    CK(cudaMemcpyAsync(c->d_V, V, c->n, cudaMemcpyDefault, st));
    CK(cudaMemcpyAsync(c->d_Yin, Y, 4 * (size_t)c->m, cudaMemcpyDefault, st));
    k_fill_i64<<<1, 32, 0, st>>>(c->d_slots + SLOT_ACC, KEY_NONE, 2);
    CK(cudaMemsetAsync(c->d_counter, 0, sizeof(unsigned), st));
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, c->d_Yin, c->d_fs);
    CK(cudaGetLastError());
    SearchArgs A = make_args(c, g, 1, 0, 0);
    CK(cudaEventRecord(c->ev0, st));
    if ((s = dispatch_step_eval(c, k, A, g, c->d_slots + SLOT_OUT, nullptr, false, st)) != LNS_OK) return s;
    CK(cudaEventRecord(c->ev1, st));
    int64_t key, fs[FS_N];
    CK(cudaMemcpyAsync(&key, c->d_slots + SLOT_OUT, 8, cudaMemcpyDeviceToHost, st));
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
    if (k >= 4) return gen_eval_all(c, k, V, fitness_out, stream);
    Geometry g;
    lns_status s = check_k(c, k, g);
    if (s != LNS_OK) return s;
    if (!V || !fitness_out) return fail(LNS_EINVAL, "null argument");
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    if ((s = grow(c->d_fit, c->fit_cap, g.M)) != LNS_OK) return s;
    CK(cudaMemcpyAsync(c->d_V, V, c->n, cudaMemcpyDefault, st));
    k_fill_i64<<<1, 32, 0, st>>>(c->d_slots + SLOT_ACC, KEY_NONE, 2);
    CK(cudaMemsetAsync(c->d_counter, 0, sizeof(unsigned), st));
    k_init<<<1, NT, 0, st>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, nullptr, c->d_fs);
    SearchArgs A = make_args(c, g, 1, 0, 0);
    A.lo = 0; A.hi = g.M;
    A.until = nullptr;
    CK(cudaEventRecord(c->ev0, st));
    if ((s = dispatch_step_eval(c, k, A, g, c->d_slots + SLOT_OUT, c->d_fit, true, st)) != LNS_OK) return s;
    CK(cudaEventRecord(c->ev1, st));
    int64_t fs[FS_N];
    CK(cudaMemcpyAsync(fs, c->d_fs, sizeof(fs), cudaMemcpyDeviceToHost, st));
    CK(cudaMemcpyAsync(fitness_out, c->d_fit, 4 * (size_t)g.M, cudaMemcpyDefault, st));
    CK(cudaStreamSynchronize(st));
    float ms = 0; cudaEventElapsedTime(&ms, c->ev0, c->ev1); c->last_ms = ms;
    if (fs[FS_ERR]) return fail(LNS_EINVAL, "V must be +-1");
    return LNS_OK;
}

lns_status lns_step_begin(lns_ctx *c, int32_t k, int64_t max_iters, int64_t tenure, uint64_t seed, const int8_t *V0,
                          int32_t flags, void *stream)
{
    Geometry g;
    lns_status s = check_k(c, k, g);
    if (s != LNS_OK) return s;
    if (max_iters < 0) return fail(LNS_EINVAL, "iters < 0");
    int64_t L;
    if ((s = resolve_tenure(g.M, tenure, L)) != LNS_OK) return s;
    if (flags & LNS_TABU_SOLUTIONS) return fail(LNS_EINVAL, "LNS_TABU_SOLUTIONS needs the persistent kernel (lns_tabu_run)");
    DeviceGuard dg(c->device);
    if ((s = search_setup(c, g, max_iters, seed, V0, (cudaStream_t)stream)) != LNS_OK) return s;
    c->step_active = true; c->step_K = k; c->step_iters = max_iters; c->step_L = L; c->step_flags = flags;
    return LNS_OK;
}

lns_status lns_step_eval(lns_ctx *c, int64_t *key_dev, void *stream)
{
    if (!c || !c->step_active || !key_dev) return fail(LNS_EINVAL, "no active stepped search");
    Geometry g;
    lns_status s = check_k(c, c->step_K, g);
    if (s != LNS_OK) return s;
    DeviceGuard dg(c->device);
    SearchArgs A = make_args(c, g, c->step_iters, c->step_L, c->step_flags);
    return dispatch_step_eval(c, c->step_K, A, g, key_dev, nullptr, false, (cudaStream_t)stream);
}

lns_status lns_step_apply(lns_ctx *c, const int64_t *key_dev, void *stream)
{
    if (!c || !c->step_active || !key_dev) return fail(LNS_EINVAL, "no active stepped search");
    Geometry g;
    lns_status s = check_k(c, c->step_K, g);
    if (s != LNS_OK) return s;
    DeviceGuard dg(c->device);
    SearchArgs A = make_args(c, g, c->step_iters, c->step_L, c->step_flags);
    return dispatch_step_apply(c->step_K, A, key_dev, (cudaStream_t)stream);
}

lns_status lns_step_end(lns_ctx *c, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit, lns_result *res, void *stream)
{
    if (!c || !c->step_active) return fail(LNS_EINVAL, "no active stepped search");
    DeviceGuard dg(c->device);
    c->step_active = false;
    return search_finish(c, V_out, trace_rank, trace_fit, res, (cudaStream_t)stream);
}

lns_status lns_tabu_run(lns_ctx *c, int32_t k, int64_t iters, int64_t tenure, uint64_t seed, const int8_t *V0,
                        int32_t flags, int8_t *V_out, int64_t *trace_rank, int64_t *trace_fit, lns_result *res,
                        void *stream)
{
    if (k >= 4) return gen_tabu_run(c, k, iters, tenure, seed, V0, flags, V_out, trace_rank, trace_fit, res, stream);
    Geometry g;
    lns_status s = check_k(c, k, g);
    if (s != LNS_OK) return s;
    if (!res) return fail(LNS_EINVAL, "res is required");
    if (iters < 0 || iters >= (int64_t)INT32_MAX) return fail(LNS_EINVAL, "iters must be in [0, 2^31)");
    int64_t L;
    if ((s = resolve_tenure(g.M, tenure, L)) != LNS_OK) return s;
    if (iters + L >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "iters + tenure >= 2^32");
    const bool sols = (flags & LNS_TABU_SOLUTIONS) != 0;
    if (sols && L < 1) return fail(LNS_EINVAL, "LNS_TABU_SOLUTIONS needs tenure >= 1");
    if (sols && c->npeers == 0 && (c->comm != nullptr || c->nparts > 1 || (flags & LNS_FORCE_STEPPED)))
        return fail(LNS_EINVAL, "LNS_TABU_SOLUTIONS needs the persistent kernel (no stepped / NCCL path)");
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    if (sols && (s = grow(c->d_ring, c->ring_cap, (size_t)L * c->NWn)) != LNS_OK) return s;
    const bool persistent = c->npeers > 0 || !(c->comm != nullptr || c->nparts > 1 || (flags & LNS_FORCE_STEPPED));
    const bool need_until = !persistent || sols || (flags & LNS_ASPIRATION) || c->no_bits;
    if ((s = search_setup(c, g, iters, seed, V0, st, need_until)) != LNS_OK) return s;
    SearchArgs A = make_args(c, g, iters, L, flags);
    bool stepped_timing = false;
    if (c->npeers > 0) {
        // device-initiated exchange: one persistent kernel per partition, meeting in the peers'
        // exchange buffers every iteration; every partition uses the same CTA count
        A.peers = c->d_peers; A.npeers = c->npeers; A.part = c->part;
        A.timeout_ns = c->peer_timeout_ms * 1000000LL;
        const uint32_t span = (uint32_t)((g.M + (uint64_t)c->nparts - 1) / (uint64_t)c->nparts);
        const int nb = search_blocks(c, span, 1);
        if (iters > 0 && (s = dispatch_search(c, k, A, g, st, nb)) != LNS_OK) return s;
    } else if (!(c->comm != nullptr || c->nparts > 1 || (flags & LNS_FORCE_STEPPED))) {
        if (iters > 0 && (s = dispatch_search(c, k, A, g, st)) != LNS_OK) return s;
    } else {
        if (c->nparts > 1 && !c->comm)
            return fail(LNS_EINVAL, "partitioned run needs a communicator or attached peers (or use the stepped API)");
        int64_t *kb = c->d_slots + SLOT_OUT;
        // one iteration: partial key of this slice, NCCL u64 MIN across the communicator, move
        auto one = [&](cudaStream_t q) -> lns_status {
            lns_status e = dispatch_step_eval(c, k, A, g, kb, nullptr, false, q);
            if (e != LNS_OK) return e;
            if (c->comm) {
                const int rc = c->nccl_allreduce(kb, kb, 1, /*ncclUint64*/ 5, /*ncclMin*/ 3, c->comm, q);
                if (rc != 0) return fail(LNS_ENCCL, "ncclAllReduce failed");
            }
            return dispatch_step_apply(k, A, kb, q);
        };
        // The loop is launch-bound for small neighbourhoods: after one direct iteration (it sets
        // the kernels' attributes) CH iterations are captured once into a CUDA graph on a private
        // stream (the kernels read the iteration from device state, so the graph replays as is)
        // and the graph is replayed on `st`; the remainder runs directly. LNS_NO_GRAPH=1 at create
        // keeps every launch direct.
        constexpr int64_t CH = 64;
        // timed as [ev0, ev2] (the direct first iteration) + [ev3, ev1] (the rest): the host-side
        // capture and instantiation in between leave the GPU idle and are not search time
        cudaGraphExec_t ge = nullptr;
        CK(cudaEventRecord(c->ev0, st));
        int64_t t = 0;
        if (iters > 0) {
            if ((s = one(st)) != LNS_OK) return s;
            t = 1;
        }
        CK(cudaEventRecord(c->ev2, st));
        if (!c->no_graph && iters - t >= CH) {
            if (!c->cap_stream) CK(cudaStreamCreateWithFlags(&c->cap_stream, cudaStreamNonBlocking));
            cudaGraph_t gr = nullptr;
            CK(cudaStreamBeginCapture(c->cap_stream, cudaStreamCaptureModeThreadLocal));
            lns_status ce = LNS_OK;
            for (int64_t q = 0; q < CH && ce == LNS_OK; q++) ce = one(c->cap_stream);
            const cudaError_t ee = cudaStreamEndCapture(c->cap_stream, &gr);
            if (ce != LNS_OK) { if (gr) cudaGraphDestroy(gr); return ce; }
            CK(ee);
            const cudaError_t ie = cudaGraphInstantiate(&ge, gr, 0);
            cudaGraphDestroy(gr);
            CK(ie);
        }
        CK(cudaEventRecord(c->ev3, st));
        stepped_timing = true;
        while (t < iters) {
            const int64_t t_prev = t;
            if (ge && iters - t >= CH) {
                const cudaError_t le = cudaGraphLaunch(ge, st);
                if (le != cudaSuccess) { cudaGraphExecDestroy(ge); return fail(LNS_ECUDA, cudaGetErrorString(le)); }
                t += CH;
            } else {
                if ((s = one(st)) != LNS_OK) { if (ge) cudaGraphExecDestroy(ge); return s; }
                t++;
            }
            if ((flags & LNS_STOP_ON_ZERO) && (t / 64) != (t_prev / 64)) {
                int64_t done;
                CK(cudaMemcpyAsync(&done, c->d_fs + FS_DONE, 8, cudaMemcpyDeviceToHost, st));
                CK(cudaStreamSynchronize(st));
                if (done) break;
            }
        }
        if (ge) cudaGraphExecDestroy(ge);
        CK(cudaEventRecord(c->ev1, st));
    }
    s = search_finish(c, V_out, trace_rank, trace_fit, res, st);
    float ms = 0, ms2 = 0;
    if (iters > 0 && stepped_timing) {
        if (cudaEventElapsedTime(&ms, c->ev0, c->ev2) == cudaSuccess &&
            cudaEventElapsedTime(&ms2, c->ev3, c->ev1) == cudaSuccess)
            c->last_ms = (double)ms + (double)ms2;
    } else if (iters > 0 && cudaEventElapsedTime(&ms, c->ev0, c->ev1) == cudaSuccess) {
        c->last_ms = ms;
    }
    cudaGetLastError();
    return s;
}

lns_status lns_tabu_run_batch(lns_ctx *c, int32_t k, int32_t R, int64_t iters, int64_t tenure, uint64_t seed,
                              const int8_t *V0, int32_t flags, int8_t *V_out, lns_result *res, void *stream)
{
    if (k >= 4) return gen_tabu_run_batch(c, k, R, iters, tenure, seed, V0, flags, V_out, res, stream);
    Geometry g;
    lns_status s = check_k(c, k, g);
    if (s != LNS_OK) return s;
    if (!res || R < 0) return fail(LNS_EINVAL, "bad argument");
    if (iters < 0 || iters >= (int64_t)INT32_MAX) return fail(LNS_EINVAL, "iters must be in [0, 2^31)");
    int64_t L;
    if ((s = resolve_tenure(g.M, tenure, L)) != LNS_OK) return s;
    if (iters + L >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "iters + tenure >= 2^32");
    const bool sols = (flags & LNS_TABU_SOLUTIONS) != 0;
    if (sols && L < 1) return fail(LNS_EINVAL, "LNS_TABU_SOLUTIONS needs tenure >= 1");
    if (R == 0) return LNS_OK;
    DeviceGuard dg(c->device);
    cudaStream_t st = (cudaStream_t)stream;
    // start vectors: given (validated) or drawn from seed_r = splitmix64(seed + r) (reading R12)
    const int n = c->n;
    std::vector<int8_t> hv((size_t)R * n);
    if (V0) {
        // ordered after the caller's work on `stream` (a device V0 may still be being written there)
        CK(cudaMemcpyAsync(hv.data(), V0, hv.size(), cudaMemcpyDefault, st));
        CK(cudaStreamSynchronize(st));
        for (int8_t v : hv)
            if (v != 1 && v != -1) return fail(LNS_EINVAL, "V0 entries must be +1 or -1");
    } else {
        for (int r = 0; r < R; r++) {
            uint64_t sr = seed + (uint64_t)r;
            vector_from_seed(n, splitmix64_next(sr), hv.data() + (size_t)r * n);
        }
    }
    // With a communicator attached (lns_attach_comm / lns_comm_init_rank) the restarts are sharded:
    // restart r runs on rank r mod world (the 50-run protocol of PAPER.md:250-253
    // spread over GPUs), and the results are gathered on every rank by one NCCL sum of the
    // zero-padded result arrays (each restart has exactly one owner). No per-iteration collective.
    const int R_all = R;
    const bool shard = c->comm && c->nparts > 1;
    std::vector<int> mine;
    for (int r = 0; r < R_all; r++)
        if (!shard || r % c->nparts == c->part) mine.push_back(r);
    if (shard) {
        std::vector<int8_t> hl(mine.size() * (size_t)n);
        for (size_t q = 0; q < mine.size(); q++)
            memcpy(hl.data() + q * n, hv.data() + (size_t)mine[q] * n, n);
        hv.swap(hl);
        R = (int)mine.size();
    }
    std::vector<int64_t> hres((size_t)R * FS_N);
    std::vector<uint32_t> hvo((size_t)R * c->NWn);
    if (R > 0) {
    // Schedule: up to two phases, k1 rounds of G1 concurrent searches on
    // SMs / G1 CTAs each, then the R2 = R - k1 G1 remaining searches at once on SMs / R2 CTAs each,
    // minimising the makespan under the iteration-time model
    //   T(nb) = (2 + 7.5e-4 m n) us + 1.45e-5 us * M (m + 32) / nb
    // (a per-iteration cost of every CTA: plan build, exchange, move; plus the evaluation spread
    // over nb SMs; fitted on C2-C4 batches of 50, nb = 2..14). The second phase fills the SMs the
    // rounds of the first would leave idle (50 searches on 148 SMs: 37 x 4 CTAs, then 13 x 11).
    const int SMs = c->numSMs;
    const double work = 1.45e-5 * (double)g.M * (double)(c->m + 32);
    const double fixed = 2.0 + 7.5e-4 * (double)c->m * (double)c->n;
    auto T = [&](int nbq) { return fixed + work / nbq; };
    const int budget = c->smemOptin - 1024;
    // a global tabu state per group (unless the slice fits in shared memory), capped at 8 GiB in
    // total: a bitmap (+ ring) in bits_mode, else a u32 until[] per rank
    const bool bits = !c->no_bits && !sols && !(flags & LNS_ASPIRATION);
    const int64_t per_group = bits ? 4 * (((int64_t)g.M + 31) / 32) + (L > 0 && L < iters ? 4 * L : 0) : 4LL * g.M;
    const int64_t cap_groups = std::max<int64_t>(1, (8LL << 30) / std::max<int64_t>(per_group, 1));
    // LNS_TABU_SOLUTIONS: a global until[] and a visited ring per group, 8 GiB in total at most
    const int64_t cap_sol = std::max<int64_t>(1, (8LL << 30) / (4LL * ((int64_t)g.M + L * c->NWn)));
    auto fits = [&](int groups, int nb_min) {
        if (sols) return groups <= cap_sol;
        const uint64_t slice = ((uint64_t)g.M + nb_min - 1) / nb_min + 64;
        return g.smem_eval + 4 * slice <= (size_t)budget || groups <= cap_groups;
    };
    int G1 = 1, k1 = R, R2 = 0;
    if (c->blocks_override > 0) {
        G1 = std::min(R, std::max(1, SMs / c->blocks_override));
        k1 = (R + G1 - 1) / G1;
    } else {
        double best = 1e300;
        for (int q = 1; q <= std::min<int>(R, SMs); q++) {
            const int nbq = SMs / q;
            for (int kq = R / q; kq >= 0; kq--) {
                const int rem = R - kq * q;
                if (rem > SMs) break;
                const int nbr = rem > 0 ? SMs / rem : nbq;
                if (!fits((kq > 0 ? q : 0) + rem, std::min(kq > 0 ? nbq : nbr, nbr))) continue;
                const double mk = kq * T(nbq) + (rem > 0 ? T(nbr) : 0.0);
                if (mk < best * 0.999) { best = mk; G1 = q; k1 = kq; R2 = rem; }
            }
        }
        if (best >= 1e300) { G1 = 1; k1 = R; R2 = 0; }  // (only the 8 GiB cap can force this)
    }
    SearchArgs phases;
    int nph = 0, ngroups = 0, grid = 0, nb_min = SMs, r0 = 0;
    auto add_phase = [&](int Gq, int nbq, int Rq) {
        phases.phG[nph] = Gq; phases.phnb[nph] = nbq; phases.phgb[nph] = ngroups;
        phases.phr0[nph] = r0; phases.phR[nph] = Rq;
        ngroups += Gq; grid = std::max(grid, Gq * nbq); nb_min = std::min(nb_min, nbq); r0 += Rq; nph++;
    };
    if (c->blocks_override > 0) add_phase(G1, std::min(c->blocks_override, SMs), R);
    else {
        if (k1 > 0) add_phase(G1, SMs / G1, k1 * G1);
        if (R2 > 0) add_phase(R2, SMs / R2, R2);
    }
    if ((s = grow(c->d_V0s, c->v0s_cap, hv.size())) != LNS_OK) return s;
    if ((s = grow(c->d_res, c->res_cap, (size_t)R * FS_N)) != LNS_OK) return s;
    if ((s = grow(c->d_vouts, c->vouts_cap, (size_t)R * c->NWn)) != LNS_OK) return s;
    if ((s = grow(c->d_gslots, c->gslots_cap, (size_t)ngroups * 64)) != LNS_OK) return s;
    if (sols && (s = grow(c->d_ring, c->ring_cap, (size_t)ngroups * L * c->NWn)) != LNS_OK) return s;
    CK(cudaMemcpyAsync(c->d_V0s, hv.data(), hv.size(), cudaMemcpyHostToDevice, st));
    const int savep = c->part, saven = c->nparts;
    c->part = 0; c->nparts = 1;
    SearchArgs A = make_args(c, g, iters, L, flags);
    c->part = savep; c->nparts = saven;
    A.R = R; A.V0s = c->d_V0s; A.res = c->d_res; A.vouts = c->d_vouts;
    A.ring = c->d_ring;
    A.trace_r = nullptr; A.trace_f = nullptr;
    A.nph = nph;
    for (int q = 0; q < nph; q++) {
        A.phG[q] = phases.phG[q]; A.phnb[q] = phases.phnb[q]; A.phgb[q] = phases.phgb[q];
        A.phr0[q] = phases.phr0[q]; A.phR[q] = phases.phR[q];
    }
    switch (k) {
    case 1: s = launch_batch<1>(c, A, g, grid, ngroups, nb_min, c->d_gslots, st); break;
    case 2: s = launch_batch<2>(c, A, g, grid, ngroups, nb_min, c->d_gslots, st); break;
    default: s = launch_batch<3>(c, A, g, grid, ngroups, nb_min, c->d_gslots, st); break;
    }
    if (s != LNS_OK) return s;
    CK(cudaMemcpyAsync(hres.data(), c->d_res, hres.size() * 8, cudaMemcpyDeviceToHost, st));
    CK(cudaMemcpyAsync(hvo.data(), c->d_vouts, hvo.size() * 4, cudaMemcpyDeviceToHost, st));
    CK(cudaStreamSynchronize(st));
    float ms = 0;
    if (cudaEventElapsedTime(&ms, c->ev0, c->ev1) == cudaSuccess) c->last_ms = ms;
    } else {
        c->last_ms = 0.0;
    }
    if (shard) {  // gather: zero-padded full arrays, one owner per restart, NCCL sum
        std::vector<int64_t> fres((size_t)R_all * FS_N, 0);
        std::vector<uint32_t> fvo((size_t)R_all * c->NWn, 0u);
        for (size_t q = 0; q < mine.size(); q++) {
            memcpy(fres.data() + (size_t)mine[q] * FS_N, hres.data() + q * FS_N, 8 * FS_N);
            memcpy(fvo.data() + (size_t)mine[q] * c->NWn, hvo.data() + q * c->NWn, 4 * (size_t)c->NWn);
        }
        if ((s = grow(c->d_res, c->res_cap, fres.size())) != LNS_OK) return s;
        if ((s = grow(c->d_vouts, c->vouts_cap, fvo.size())) != LNS_OK) return s;
        CK(cudaMemcpyAsync(c->d_res, fres.data(), fres.size() * 8, cudaMemcpyHostToDevice, st));
        CK(cudaMemcpyAsync(c->d_vouts, fvo.data(), fvo.size() * 4, cudaMemcpyHostToDevice, st));
        if (c->nccl_allreduce(c->d_res, c->d_res, fres.size(), /*ncclInt64*/ 4, /*ncclSum*/ 0, c->comm, st) != 0 ||
            c->nccl_allreduce(c->d_vouts, c->d_vouts, fvo.size(), /*ncclUint32*/ 3, /*ncclSum*/ 0, c->comm, st) != 0)
            return fail(LNS_ENCCL, "ncclAllReduce (restart gather) failed");
        CK(cudaMemcpyAsync(fres.data(), c->d_res, fres.size() * 8, cudaMemcpyDeviceToHost, st));
        CK(cudaMemcpyAsync(fvo.data(), c->d_vouts, fvo.size() * 4, cudaMemcpyDeviceToHost, st));
        CK(cudaStreamSynchronize(st));
        hres.swap(fres);
        hvo.swap(fvo);
        R = R_all;
    }
    for (int r = 0; r < R; r++) {
        const int64_t *o = hres.data() + (size_t)r * FS_N;
        if (o[FS_ERR] == 4) return fail(LNS_EPEER, "a CTA of the grid did not reach the exchange in time");
        if (o[FS_ERR] == 2) return fail(LNS_ENOADMISSIBLE, "no admissible move");
        res[r].iters_done = o[FS_T]; res[r].final_f = o[FS_F]; res[r].best_f = o[FS_BEST];
        res[r].best_iter = o[FS_BESTIT]; res[r].first_zero_iter = o[FS_ZERO];
        res[r].solved = o[FS_BEST] == 0; res[r].reserved = 0;
    }
    if (V_out) {
        std::vector<int8_t> ho((size_t)R * n);
        for (int r = 0; r < R; r++)
            for (int i = 0; i < n; i++)
                ho[(size_t)r * n + i] = ((hvo[(size_t)r * c->NWn + i / 32] >> (i % 32)) & 1) ? -1 : 1;
        CK(cudaMemcpyAsync(V_out, ho.data(), ho.size(), cudaMemcpyDefault, st));
        CK(cudaStreamSynchronize(st));
    }
    return LNS_OK;
}

#ifdef LNS_PHASE_TIMING
// Profiling build only: per-phase cycle sums of thread 0 of every CTA since the last call (PH()).
lns_status lns_debug_phases(unsigned long long *out8)
{
    CK(cudaMemcpyFromSymbol(out8, g_ph, sizeof(unsigned long long) * NPH));
    unsigned long long z[NPH] = {0};
    CK(cudaMemcpyToSymbol(g_ph, z, sizeof(z)));
    return LNS_OK;
}
#endif

// Undocumented debug export (tests/tools only): plan of V for neighbourhood k, see k_debug_plan.
lns_status lns_debug_plan(lns_ctx *c, int32_t k, const int8_t *V, int32_t *out_host, int64_t cap)
{
    Geometry g;
    lns_status s = check_k(c, k, g);
    if (s != LNS_OK) return s;
    DeviceGuard dg(c->device);
    int32_t *d_out = nullptr;
    CK(cudaMalloc(&d_out, cap * 4));
    CK(cudaMemcpy(c->d_V, V, c->n, cudaMemcpyDefault));
    k_init<<<1, NT>>>(dev_inst(c), c->d_V, c->d_vb, c->d_Y, nullptr, c->d_fs);
    SearchArgs A = make_args(c, g, 1, 0, 0);
    const int sm = (int)g.smem_eval;
    if (k == 1) { cudaFuncSetAttribute(k_debug_plan<1>, cudaFuncAttributeMaxDynamicSharedMemorySize, sm); k_debug_plan<1><<<1, NT, sm>>>(A, d_out); }
    else if (k == 2) { cudaFuncSetAttribute(k_debug_plan<2>, cudaFuncAttributeMaxDynamicSharedMemorySize, sm); k_debug_plan<2><<<1, NT, sm>>>(A, d_out); }
    else { cudaFuncSetAttribute(k_debug_plan<3>, cudaFuncAttributeMaxDynamicSharedMemorySize, sm); k_debug_plan<3><<<1, NT, sm>>>(A, d_out); }
    CK(cudaMemcpy(out_host, d_out, cap * 4, cudaMemcpyDeviceToHost));
    cudaFree(d_out);
    return LNS_OK;
}

lns_status lns_unrank(int32_t n, int32_t k, const int64_t *ranks, int64_t count, int32_t *out, void *stream)
{
    if (k >= 4 && k <= KG_MAX && n >= k) {  // generic-k unranking (k_gen's), count x k entries
        if (count < 0 || (count > 0 && (!ranks || !out))) return fail(LNS_EINVAL, "bad buffers");
        const int64_t Mk = comb_k(n, k);
        if (Mk < 0 || Mk >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "C(n,k) >= 2^32-1");
        if (count == 0) return LNS_OK;
        cudaStream_t st = (cudaStream_t)stream;
        int64_t *d_r = nullptr;
        int32_t *d_o = nullptr, *d_bad = nullptr;
        if (cudaMalloc(&d_r, count * 8) != cudaSuccess || cudaMalloc(&d_o, count * 4 * k) != cudaSuccess ||
            cudaMalloc(&d_bad, 4) != cudaSuccess) {
            cudaFree(d_r); cudaFree(d_o); cudaGetLastError();
            return fail(LNS_ENOMEM, "cudaMalloc failed");
        }
        int bad = 0;
        cudaMemcpyAsync(d_r, ranks, count * 8, cudaMemcpyDefault, st);
        cudaMemsetAsync(d_bad, 0, 4, st);
        const int blocks = (int)std::min<int64_t>((count + 255) / 256, 4096);
        k_unrank_gen<<<blocks, 256, 8 * (size_t)(n + 1) * (k + 1), st>>>(n, k, (uint32_t)Mk, d_r, count, d_o, d_bad);
        cudaMemcpyAsync(out, d_o, count * 4 * k, cudaMemcpyDefault, st);
        cudaMemcpyAsync(&bad, d_bad, 4, cudaMemcpyDeviceToHost, st);
        const cudaError_t e = cudaStreamSynchronize(st);
        cudaFree(d_r); cudaFree(d_o); cudaFree(d_bad);
        if (e != cudaSuccess) return fail(LNS_ECUDA, cudaGetErrorString(e));
        if (bad) return fail(LNS_EINVAL, "rank out of range");
        return LNS_OK;
    }
    if (k < 1 || k > 3 || n < k) return fail(LNS_EINVAL, "bad n/k");
    if (count < 0 || (count > 0 && (!ranks || !out))) return fail(LNS_EINVAL, "bad buffers");
    const int64_t Mk = comb_k(n, k);
    if (Mk >= (int64_t)UINT32_MAX) return fail(LNS_ERANGE, "C(n,k) >= 2^32-1");
    if (count == 0) return LNS_OK;
    cudaStream_t st = (cudaStream_t)stream;
    int64_t *d_r = nullptr;
    int32_t *d_o = nullptr, *d_bad = nullptr;
    if (cudaMalloc(&d_r, count * 8) != cudaSuccess || cudaMalloc(&d_o, count * 12) != cudaSuccess ||
        cudaMalloc(&d_bad, 4) != cudaSuccess) {
        cudaFree(d_r); cudaFree(d_o); cudaGetLastError();
        return fail(LNS_ENOMEM, "cudaMalloc failed");
    }
    int bad = 0;
    cudaMemcpyAsync(d_r, ranks, count * 8, cudaMemcpyDefault, st);
    cudaMemsetAsync(d_bad, 0, 4, st);
    const int blocks = (int)std::min<int64_t>((count + 255) / 256, 4096);
    const size_t tsm = 8 * (size_t)n;
    // both the hot-path (table) unranking and the 64-bit reference; they must agree
    int32_t *d_o2 = nullptr;
    if (cudaMalloc(&d_o2, count * 12) != cudaSuccess) { cudaFree(d_r); cudaFree(d_o); cudaFree(d_bad); cudaGetLastError(); return fail(LNS_ENOMEM, "cudaMalloc failed"); }
    for (int tab = 0; tab < 2; tab++) {
        int32_t *o = tab ? d_o : d_o2;
        if (k == 1) k_unrank<1><<<blocks, 256, tsm, st>>>(n, (uint32_t)Mk, d_r, count, o, d_bad, tab);
        else if (k == 2) k_unrank<2><<<blocks, 256, tsm, st>>>(n, (uint32_t)Mk, d_r, count, o, d_bad, tab);
        else k_unrank<3><<<blocks, 256, tsm, st>>>(n, (uint32_t)Mk, d_r, count, o, d_bad, tab);
    }
    std::vector<int32_t> h1((size_t)count * 3), h2((size_t)count * 3);
    cudaMemcpyAsync(h1.data(), d_o, count * 12, cudaMemcpyDeviceToHost, st);
    cudaMemcpyAsync(h2.data(), d_o2, count * 12, cudaMemcpyDeviceToHost, st);
    cudaMemcpyAsync(out, d_o, count * 12, cudaMemcpyDefault, st);
    cudaMemcpyAsync(&bad, d_bad, 4, cudaMemcpyDeviceToHost, st);
    const cudaError_t e = cudaStreamSynchronize(st);
    cudaFree(d_r); cudaFree(d_o); cudaFree(d_o2); cudaFree(d_bad);
    if (e != cudaSuccess) return fail(LNS_ECUDA, cudaGetErrorString(e));
    if (bad) return fail(LNS_EINVAL, "rank out of range");
    if (h1 != h2) return fail(LNS_ECUDA, "table and reference unranking disagree");
    return LNS_OK;
}

}  // extern "C"

#include "bqp.cuh"  // second binary fitness (UBQP), DESIGN.md §5.13

// int_peaks.cu -- measured integer-pipe peaks of this GPU ("the integer peak is
// measured, not assumed"). For every instruction class the tabu-search record loop issues (LOP3,
// IADD3, IMAD, POPC, PRMT, SHF funnel, VABSDIFF4, IDP.2A, LDS), a kernel runs long unrolled
// streams of that instruction over 8 independent chains per thread, 1024 threads per CTA,
// 2 CTAs per SM, and reports lanes per clock per SM from clock64() (SM cycles, so the figure
// is clock independent). "mix_lop3_imad" alternates the ALU and FMA pipes (the issue limit:
// one warp instruction per clock per SMSP = 128 lanes/clk/SM); "record_mix" is the instruction
// mix of one record of the packed evaluation loop (3 LOP3 + 3 POPC + 3 IMAD + PRMT + IDP +
// VABSDIFF4 + SHF).
//
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o int_peaks int_peaks.cu && ./int_peaks
// prints one JSON object.
#include <cstdio>
#include <cuda_runtime.h>

#define NCH 8
#define REP 256
#define NT 1024

struct Out {
    unsigned long long t0, t1;  // clock64() at start / end (SM cycles; one clock per SM)
    unsigned smid, sink;
};

template <int OP>
__device__ __forceinline__ void step(unsigned (&x)[NCH], unsigned k1, unsigned k2)
{
#pragma unroll
    for (int c = 0; c < NCH; c++) {
        unsigned a = x[c];
        if (OP == 0) asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(a) : "r"(k1), "r"(k2));
        if (OP == 1) asm volatile("add.u32 %0, %0, %1;" : "+r"(a) : "r"(k1));
        if (OP == 2) asm volatile("mad.lo.u32 %0, %0, %1, %2;" : "+r"(a) : "r"(k1), "r"(k2));
        if (OP == 3) asm volatile("popc.b32 %0, %0;" : "+r"(a));
        if (OP == 4) asm volatile("prmt.b32 %0, %0, %1, %2;" : "+r"(a) : "r"(k1), "r"(k2));
        if (OP == 5) asm volatile("shf.r.wrap.b32 %0, %0, %1, %2;" : "+r"(a) : "r"(k1), "r"(k2));
        if (OP == 6) asm volatile("vabsdiff4.u32.u32.u32.add %0, %0, %1, %2;" : "+r"(a) : "r"(k1), "r"(k2));
        if (OP == 7) asm volatile("dp2a.lo.u32.u32 %0, %0, %1, %2;" : "+r"(a) : "r"(k1), "r"(k2));
        if (OP == 8) {  // alternate ALU (LOP3) and FMA (IMAD) pipes
            if (c & 1) asm volatile("mad.lo.u32 %0, %0, %1, %2;" : "+r"(a) : "r"(k1), "r"(k2));
            else asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(a) : "r"(k1), "r"(k2));
        }
        x[c] = a;
    }
}

// one record of the packed loop per chain pair: 3 (LOP3, POPC, IMAD) + PRMT + IDP + VABSDIFF4 + SHF
__device__ __forceinline__ void record(unsigned (&x)[NCH], unsigned k1, unsigned k2)
{
#pragma unroll
    for (int c = 0; c < NCH; c += 2) {
        unsigned w = x[c], f = x[c + 1], p, hb;
#pragma unroll
        for (int q = 0; q < 3; q++) {
            asm volatile("lop3.b32 %0, %1, %2, %3, 0xc0;" : "=r"(p) : "r"(w), "r"(k1), "r"(k2));
            asm volatile("popc.b32 %0, %0;" : "+r"(p));
            asm volatile("mad.lo.u32 %0, %1, 255, %0;" : "+r"(w) : "r"(p));
        }
        asm volatile("prmt.b32 %0, %1, 0, %2;" : "=r"(hb) : "r"(w), "r"(k2));
        asm volatile("dp2a.lo.u32.u32 %0, %1, %2, %0;" : "+r"(f) : "r"(k2), "r"(hb));
        asm volatile("vabsdiff4.u32.u32.u32.add %0, %1, %2, %0;" : "+r"(f) : "r"(hb), "r"(k1));
        asm volatile("shf.r.wrap.b32 %0, %0, %1, %2;" : "+r"(w) : "r"(k1), "r"(k2));
        x[c] = w; x[c + 1] = f;
    }
}

template <int OP>
__global__ void __launch_bounds__(NT, 2) k_peak(Out *out, unsigned seed, int iters)
{
    unsigned x[NCH];
#pragma unroll
    for (int c = 0; c < NCH; c++) x[c] = seed * (threadIdx.x + 7 * c + 1);
    const unsigned k1 = seed ^ 0x5bd1e995u, k2 = seed + 0x27d4eb2du;
    __syncthreads();
    const unsigned long long t0 = clock64();
    for (int i = 0; i < iters; i++) {
#pragma unroll
        for (int r = 0; r < REP; r++) {
            if (OP == 9) record(x, k1, k2);
            else step<OP>(x, k1, k2);
        }
    }
    __syncthreads();
    const unsigned long long t1 = clock64();
    unsigned s = 0;
#pragma unroll
    for (int c = 0; c < NCH; c++) s ^= x[c];
    if (threadIdx.x == 0) {
        unsigned sm;
        asm volatile("mov.u32 %0, %%smid;" : "=r"(sm));
        out[blockIdx.x].t0 = t0; out[blockIdx.x].t1 = t1; out[blockIdx.x].smid = sm;
    }
    if (s == 0x12345678u) out[blockIdx.x].sink = s;
}

template <int OP>
double run(const char *name, int sms, Out *d, double inst_per_chain_step, bool first)
{
    const int grid = 2 * sms, iters = 40;
    k_peak<OP><<<grid, NT>>>(d, 3u, 2);  // warm-up
    cudaDeviceSynchronize();
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0); cudaEventCreate(&e1);
    cudaEventRecord(e0);
    k_peak<OP><<<grid, NT>>>(d, 3u, iters);
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms = 0;
    cudaEventElapsedTime(&ms, e0, e1);
    Out *h = new Out[grid];
    cudaMemcpy(h, d, sizeof(Out) * grid, cudaMemcpyDeviceToHost);
    // per SM: busy cycles = last end - first start over its CTAs (same SM clock); lanes per SM
    // from the CTAs it ran. Rate = sum lanes / sum busy cycles over the SMs.
    const double lanes_cta = (double)NT * iters * REP * NCH * inst_per_chain_step;
    double busy = 0, lanes = 0;
    for (int smx = 0; smx < 1024; smx++) {
        unsigned long long a = ~0ull, b = 0;
        int c = 0;
        for (int q = 0; q < grid; q++)
            if ((int)h[q].smid == smx) { a = h[q].t0 < a ? h[q].t0 : a; b = h[q].t1 > b ? h[q].t1 : b; c++; }
        if (c) { busy += (double)(b - a); lanes += c * lanes_cta; }
    }
    delete[] h;
    const double per_clk = lanes / busy;
    const double cyc = busy / sms;
    const double per_s = lanes / (ms * 1e-3);
    printf("%s\"%s\": {\"lanes_per_clk_per_sm\": %.2f, \"warp_inst_per_clk_per_smsp\": %.3f, "
           "\"chip_lane_ops_per_s\": %.4e, \"sm_mhz_implied\": %.0f}",
           first ? "" : ", ", name, per_clk, per_clk / 128.0, per_s, cyc / (ms * 1e3));
    return per_clk;
}

int main()
{
    int dev = 0, sms = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    cudaDeviceProp p;
    cudaGetDeviceProperties(&p, dev);
    Out *d = nullptr;
    cudaMalloc(&d, sizeof(Out) * 2 * sms);
    printf("{\"gpu\": \"%s\", \"sms\": %d, \"threads_per_sm\": %d, \"chains_per_thread\": %d, \"peaks\": {", p.name,
           sms, 2 * NT, NCH);
    run<0>("lop3", sms, d, 1.0, true);
    run<1>("iadd3", sms, d, 0.5, false);  // ptxas fuses two dependent adds into one IADD3
    run<2>("imad", sms, d, 1.0, false);
    run<3>("popc", sms, d, 1.0, false);
    run<4>("prmt", sms, d, 1.0, false);
    run<5>("shf_funnel", sms, d, 1.0, false);
    run<6>("vabsdiff4", sms, d, 1.0, false);
    run<7>("idp_2a", sms, d, 1.0, false);
    run<8>("mix_lop3_imad", sms, d, 1.0, false);
    run<9>("record_mix", sms, d, 13.0 / 2.0, false);  // 13 instructions per chain pair
    printf("}}\n");
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) { fprintf(stderr, "CUDA error: %s\n", cudaGetErrorString(e)); return 1; }
    return 0;
}

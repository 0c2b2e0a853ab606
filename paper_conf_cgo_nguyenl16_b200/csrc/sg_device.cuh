// sg_device.cuh -- hand-written sm_100a device code of the stream-graph executor.
//
// Embedded into libsg.so at build time and handed to NVRTC together with the
// per-partition kernel that sg_codegen.cpp generates ("the GPU code generator
// ... generates the CUDA code").  One partition = one kernel
// (PAPER.md:553-555, 709).
//
// Contents:
//   1. work functions, one per filter kind: the filter body executed for ONE
//      firing on values held in registers.  Semantics = include/sg.h (readings
//      of SURVEY.md 8(c)-3).  Compiled with --fmad=false, no fast math, IEEE
//      division/sqrt: every multiply-add written as fmaf() below is one FFMA,
//      every other product one FMUL.
//   2. tile movers: coalesced, vectorised global<->shared copies used by the
//      generated kernels (the "data transfer" role of the paper's DT threads,
//      PAPER.md:220-228, done here by all threads between compute phases or by
//      the TMA engine).
//   3. TMA / mbarrier helpers (cp.async.bulk.tensor) for row-regular tiles.
#pragma once

#define SG_DEV __device__ __forceinline__

typedef int sg_i32;
typedef unsigned int sg_u32;
typedef long long sg_i64;

// ---------------------------------------------------------------- 1. work
template <typename T>
SG_DEV void sg_work_identity(const T (&x)[1], T (&y)[1]) { y[0] = x[0]; }

// FIR: acc = 0; acc = fma(peek(i), c[i], acc), i = 0..L-1  (taps oldest first)
template <int PEEK, int L>
SG_DEV void sg_work_fir(const float (&x)[PEEK], float (&y)[1], const float* __restrict__ c) {
    float acc = 0.0f;
#pragma unroll
    for (int i = 0; i < L; i++) acc = fmaf(x[i], c[i], acc);
    y[0] = acc;
}

template <typename T, int M>
SG_DEV void sg_work_decimate(const T (&x)[M], T (&y)[1]) { y[0] = x[0]; }

template <typename T, int M>
SG_DEV void sg_work_expand(const T (&x)[1], T (&y)[M]) {
    y[0] = x[0];
#pragma unroll
    for (int i = 1; i < M; i++) y[i] = (T)0;
}

// CompareExchange: (min, max) if up, (max, min) otherwise; ties keep k1 first.
template <typename T, bool UP>
SG_DEV void sg_work_compare_exchange(const T (&x)[2], T (&y)[2]) {
    const T k1 = x[0], k2 = x[1];
    const bool le = k1 <= k2;
    const T lo = le ? k1 : k2, hi = le ? k2 : k1;
    if (UP) { y[0] = lo; y[1] = hi; } else { y[0] = hi; y[1] = lo; }
}

// FFTReorderSimple(n): complex items with even index first, then odd.
template <int N>
SG_DEV void sg_work_fft_reorder(const float (&x)[2 * N], float (&y)[2 * N]) {
    int o = 0;
#pragma unroll
    for (int i = 0; i < N; i += 2) { y[o++] = x[2 * i]; y[o++] = x[2 * i + 1]; }
#pragma unroll
    for (int i = 1; i < N; i += 2) { y[o++] = x[2 * i]; y[o++] = x[2 * i + 1]; }
}

// CombineDFT(j): j/2 butterflies pairing complex k and k + j/2, w_k = e^{-2 pi i k / j}.
template <int J>
SG_DEV void sg_work_combine_dft(const float (&x)[2 * J], float (&y)[2 * J], const float* __restrict__ wr,
                                const float* __restrict__ wi) {
#pragma unroll
    for (int k = 0; k < J / 2; k++) {
        const float y0r = x[2 * k], y0i = x[2 * k + 1];
        const float y1r = x[2 * (k + J / 2)], y1i = x[2 * (k + J / 2) + 1];
        const float tr = fmaf(y1r, wr[k], -(y1i * wi[k]));
        const float ti = fmaf(y1r, wi[k], y1i * wr[k]);
        y[2 * k] = y0r + tr;
        y[2 * k + 1] = y0i + ti;
        y[2 * (k + J / 2)] = y0r - tr;
        y[2 * (k + J / 2) + 1] = y0i - ti;
    }
}

// FMDemodulator: (float)(gain * atan((double)(x0 * x1))), fp64 atan.
SG_DEV void sg_work_fm_demod(const float (&x)[2], float (&y)[1], float gain) {
    const float p = x[0] * x[1];
    y[0] = (float)((double)gain * atan((double)p));
}

// fp32 variant (SG_FM_F32=1 at plan time): atanf (<= 2 ulp), within the fp32 tolerance, not bit-exact
SG_DEV void sg_work_fm_demod_f32(const float (&x)[2], float (&y)[1], float gain) {
    const float p = x[0] * x[1];
    y[0] = gain * atanf(p);
}

SG_DEV void sg_work_subtract(const float (&x)[2], float (&y)[1]) { y[0] = x[1] - x[0]; }

SG_DEV void sg_work_amplify(const float (&x)[1], float (&y)[1], float k) { y[0] = x[0] * k; }

template <int N>
SG_DEV void sg_work_add(const float (&x)[N], float (&y)[1]) {
    float s = 0.0f;
#pragma unroll
    for (int i = 0; i < N; i++) s = s + x[i];
    y[0] = s;
}
template <int N>
SG_DEV void sg_work_add(const int (&x)[N], int (&y)[1]) {  // two's-complement wrap
    sg_u32 s = 0u;
#pragma unroll
    for (int i = 0; i < N; i++) s = s + (sg_u32)x[i];
    y[0] = (int)s;
}

// one complex multiply-accumulate, fixed order (SG_K_BEAM_FIR / SG_K_BEAMFORM)
SG_DEV void sg_cmac(float& re, float& im, float xr, float xi, float wr, float wi) {
    re = fmaf(xr, wr, re);
    re = fmaf(-xi, wi, re);
    im = fmaf(xr, wi, im);
    im = fmaf(xi, wr, im);
}

template <int NC>
SG_DEV void sg_work_beamform(const float (&x)[2 * NC], float (&y)[2], const float* __restrict__ wr,
                             const float* __restrict__ wi) {
    float re = 0.0f, im = 0.0f;
#pragma unroll
    for (int c = 0; c < NC; c++) sg_cmac(re, im, x[2 * c], x[2 * c + 1], wr[c], wi[c]);
    y[0] = re;
    y[1] = im;
}

SG_DEV void sg_work_multiply(const float (&x)[2], float (&y)[1]) { y[0] = __fmul_rn(x[0], x[1]); }
// DES bit kinds (include/sg.h table); items are int32, bits are x & 1
template <int N>
SG_DEV void sg_work_xor(const int (&x)[2 * N], int (&y)[N]) {
#pragma unroll
    for (int i = 0; i < N; i++) y[i] = x[i] ^ x[N + i];
}
// S-box as four 64-entry truth tables: output bit i (most significant first) = (M_i >> idx) & 1,
// idx = 16 * (2 b0 + b5) + (8 b1 + 4 b2 + 2 b3 + b4) (FIPS 46-3 row / column rule)
SG_DEV void sg_work_sbox(const int (&x)[6], int (&y)[4], unsigned long long m0, unsigned long long m1,
                         unsigned long long m2, unsigned long long m3) {
    const unsigned idx = ((x[0] & 1u) << 5) | ((x[5] & 1u) << 4) | ((x[1] & 1u) << 3) | ((x[2] & 1u) << 2) |
                         ((x[3] & 1u) << 1) | (x[4] & 1u);
    y[0] = (int)((m0 >> idx) & 1ull);
    y[1] = (int)((m1 >> idx) & 1ull);
    y[2] = (int)((m2 >> idx) & 1ull);
    y[3] = (int)((m3 >> idx) & 1ull);
}
SG_DEV void sg_work_into_bits(const int (&x)[1], int (&y)[32]) {
#pragma unroll
    for (int k = 0; k < 32; k++) y[k] = (int)(((unsigned)x[0] >> (31 - k)) & 1u);
}
SG_DEV void sg_work_bits_to_int(const int (&x)[32], int (&y)[1]) {
    unsigned v = 0u;
#pragma unroll
    for (int k = 0; k < 32; k++) v |= ((unsigned)x[k] & 1u) << (31 - k);
    y[0] = (int)v;
}
// bitslice mode: any 3-input boolean function in one LOP3 (LUT index a<<2 | b<<1 | c)
template <int LUT>
SG_DEV unsigned sg_lop3(unsigned a, unsigned b, unsigned c) {
    unsigned d;
    asm("lop3.b32 %0, %1, %2, %3, %4;" : "=r"(d) : "r"(a), "r"(b), "r"(c), "n"(LUT));
    return d;
}
// 32x32 bit-matrix transpose in registers: afterwards bit j of a[i] = bit i of the old a[j].
// Stages 16 and 8 swap whole half-words / bytes: one byte permute per output word; stages 4, 2, 1
// exchange masked bit groups.
SG_DEV void sg_transpose32(unsigned (&a)[32]) {
#pragma unroll
    for (int i = 0; i < 16; i++) {
        const unsigned x = a[i], y = a[i + 16];
        a[i] = __byte_perm(x, y, 0x5410);       // [lo16(y) | lo16(x)]
        a[i + 16] = __byte_perm(x, y, 0x7632);  // [hi16(y) | hi16(x)]
    }
#pragma unroll
    for (int i = 0; i < 32; i++) {
        if (i & 8) continue;
        const unsigned x = a[i], y = a[i + 8];
        a[i] = __byte_perm(x, y, 0x6240);       // bytes (y2, x2, y0, x0)
        a[i + 8] = __byte_perm(x, y, 0x7351);   // bytes (y3, x3, y1, x1)
    }
#pragma unroll
    for (unsigned s = 4, m = 0x0F0F0F0Fu; s > 0; s >>= 1, m ^= m << s) {
#pragma unroll
        for (int i = 0; i < 32; i++) {
            if (i & s) continue;
            const unsigned t = ((a[i] >> s) ^ a[i + s]) & m;
            a[i + s] ^= t;
            a[i] ^= t << s;
        }
    }
}
SG_DEV void sg_work_magnitude(const float (&x)[2], float (&y)[1]) {
    const float b2 = x[1] * x[1];
    y[0] = __fsqrt_rn(fmaf(x[0], x[0], b2));
}

// ------------------------------------------------------------ 2. movers
SG_DEV sg_i64 sg_fdiv(sg_i64 a, sg_i64 b) { sg_i64 q = a / b; return (a % b != 0 && ((a < 0) != (b < 0))) ? q - 1 : q; }
SG_DEV sg_i64 sg_fmod(sg_i64 a, sg_i64 b) { return a - sg_fdiv(a, b) * b; }
SG_DEV int sg_fdiv32(int a, int b) { int q = a / b; return (a % b != 0 && ((a < 0) != (b < 0))) ? q - 1 : q; }
SG_DEV int sg_fmod32(int a, int b) { return a - sg_fdiv32(a, b) * b; }

// Copy `rows` rows of R items (contiguous in global) into shared rows of stride RS.
// R % 4 == 0, RS % 4 == 0, 16-byte aligned global base: one 128-bit access per
// thread per step, consecutive threads on consecutive 16-byte chunks (coalesced).
template <typename T, int R, int RS, int NT>
SG_DEV void sg_rows_g2s_v4(const T* __restrict__ g, T* s, int rows) {
    const int nq = rows * (R / 4);
    const int4* g4 = reinterpret_cast<const int4*>(g);
#pragma unroll 4
    for (int q = threadIdx.x; q < nq; q += NT) {
        const int row = q / (R / 4), c = q - row * (R / 4);
        int4 v;
        asm volatile("ld.global.nc.L1::no_allocate.v4.s32 {%0,%1,%2,%3}, [%4];"
                     : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "l"(g4 + q));
        *reinterpret_cast<int4*>(s + row * RS + 4 * c) = v;
    }
}
template <typename T, int R, int RS, int NT>
SG_DEV void sg_rows_s2g_v4(const T* s, T* __restrict__ g, int rows) {
    const int nq = rows * (R / 4);
    int4* g4 = reinterpret_cast<int4*>(g);
#pragma unroll 4
    for (int q = threadIdx.x; q < nq; q += NT) {
        const int row = q / (R / 4), c = q - row * (R / 4);
        const int4 v = *reinterpret_cast<const int4*>(s + row * RS + 4 * c);
        asm volatile("st.global.L1::no_allocate.v4.s32 [%0], {%1,%2,%3,%4};"
                     :: "l"(g4 + q), "r"(v.x), "r"(v.y), "r"(v.z), "r"(v.w) : "memory");
    }
}
template <typename T, int R, int RS, int NT>
SG_DEV void sg_rows_g2s_v1(const T* __restrict__ g, T* s, int rows) {
    const int n = rows * R;
    for (int i = threadIdx.x; i < n; i += NT) {
        const int row = i / R, c = i - row * R;
        s[row * RS + c] = g[i];
    }
}
template <typename T, int R, int RS, int NT>
SG_DEV void sg_rows_s2g_v1(const T* s, T* __restrict__ g, int rows) {
    const int n = rows * R;
    for (int i = threadIdx.x; i < n; i += NT) {
        const int row = i / R, c = i - row * R;
        g[i] = s[row * RS + c];
    }
}

// ---------------------------------------------------- 3. TMA / mbarrier
SG_DEV sg_u32 sg_smem_addr(const void* p) { return (sg_u32)__cvta_generic_to_shared(p); }

SG_DEV void sg_mbar_init(unsigned long long* bar, int count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" :: "r"(sg_smem_addr(bar)), "r"(count));
}
SG_DEV void sg_fence_barrier_init() { asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory"); }
SG_DEV void sg_fence_proxy_async() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }

SG_DEV void sg_mbar_arrive_expect_tx(unsigned long long* bar, sg_u32 bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" :: "r"(sg_smem_addr(bar)), "r"(bytes)
                 : "memory");
}
SG_DEV void sg_mbar_arrive(unsigned long long* bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" :: "r"(sg_smem_addr(bar)) : "memory");
}
SG_DEV void sg_mbar_wait(unsigned long long* bar, sg_u32 parity) {
    asm volatile(
        "{\n"
        ".reg .pred P1;\n"
        "SG_WAIT_%=:\n"
        "mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n"
        "@!P1 bra SG_WAIT_%=;\n"
        "}\n" :: "r"(sg_smem_addr(bar)), "r"(parity) : "memory");
}

// 2-D tensor-map tile load (global -> shared), completion on `bar`.
SG_DEV void sg_tma_load_2d(void* sdst, const void* tmap, int c0, int c1, unsigned long long* bar) {
    asm volatile(
        "cp.async.bulk.tensor.2d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3}], [%4];"
        :: "r"(sg_smem_addr(sdst)), "l"(tmap), "r"(c0), "r"(c1), "r"(sg_smem_addr(bar)) : "memory");
}
// 2-D tensor-map tile store (shared -> global), bulk-group completion.
SG_DEV void sg_tma_store_2d(const void* tmap, int c0, int c1, const void* ssrc) {
    asm volatile("cp.async.bulk.tensor.2d.global.shared::cta.tile.bulk_group [%0, {%1, %2}], [%3];"
                 :: "l"(tmap), "r"(c0), "r"(c1), "r"(sg_smem_addr(ssrc)) : "memory");
}
// 1-D bulk copies (cp.async.bulk): 16-byte aligned addresses, size multiple of 16.
SG_DEV void sg_bulk_g2s(void* sdst, const void* gsrc, sg_u32 bytes, unsigned long long* bar) {
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
                 :: "r"(sg_smem_addr(sdst)), "l"(gsrc), "r"(bytes), "r"(sg_smem_addr(bar)) : "memory");
}
SG_DEV void sg_bulk_s2g(void* gdst, const void* ssrc, sg_u32 bytes) {
    asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;"
                 :: "l"(gdst), "r"(sg_smem_addr(ssrc)), "r"(bytes) : "memory");
}
SG_DEV void sg_bulk_commit() { asm volatile("cp.async.bulk.commit_group;" ::: "memory"); }
template <int N>
SG_DEV void sg_bulk_wait_read() { asm volatile("cp.async.bulk.wait_group.read %0;" :: "n"(N) : "memory"); }
template <int N>
SG_DEV void sg_bulk_wait() { asm volatile("cp.async.bulk.wait_group %0;" :: "n"(N) : "memory"); }
// 4-byte cp.async (LDGSTS) with zero fill: src_bytes = 0 writes 0 and reads nothing
// (stream positions outside [0, limit) are the zero history of the stream start).
SG_DEV void sg_cp_async4(void* sdst, const void* gsrc, sg_u32 src_bytes) {
    asm volatile("cp.async.ca.shared.global [%0], [%1], 4, %2;"
                 :: "r"(sg_smem_addr(sdst)), "l"(gsrc), "r"(src_bytes) : "memory");
}
SG_DEV void sg_cp_async16(void* sdst, const void* gsrc) {
    asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" :: "r"(sg_smem_addr(sdst)), "l"(gsrc) : "memory");
}
SG_DEV void sg_cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
SG_DEV void sg_cp_async_wait_all() { asm volatile("cp.async.wait_all;" ::: "memory"); }
SG_DEV void sg_prefetch_tmap(const void* tmap) {
    asm volatile("prefetch.tensormap [%0];" :: "l"(tmap) : "memory");
}

// Tensor-map kernel parameter (CUtensorMap is 128 bytes, 64-byte aligned).
struct __align__(64) SgTmap { unsigned long long v[16]; };

// 128B-swizzle address of 16-byte chunk `c` (0..7) of row `r` in a [rows][128 B] tile
// written by TMA with CU_TENSOR_MAP_SWIZZLE_128B (tile base 1024-byte aligned).
SG_DEV int sg_swz128(int r, int c) { return r * 128 + ((c ^ (r & 7)) << 4); }

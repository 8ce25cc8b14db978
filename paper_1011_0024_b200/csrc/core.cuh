// core.cuh — device building blocks: complex arithmetic, site-major SoA storage in the three
// precisions (P:396-424 field ordering; P:507-520 half = 16-bit fixed point with a per-site
// norm), SU(3) link reconstruction (P:475-478 two-row; reading Q6 eight-parameter).
#pragma once
#include <cuda_runtime.h>
#include <cstdint>
#include <type_traits>

namespace qx {

template <typename R>
struct Cx {
    R r, i;
};
template <typename R> __device__ __forceinline__ Cx<R> cx(R r, R i) { return Cx<R>{r, i}; }
template <typename R> __device__ __forceinline__ Cx<R> operator+(Cx<R> a, Cx<R> b) { return {a.r + b.r, a.i + b.i}; }
template <typename R> __device__ __forceinline__ Cx<R> operator-(Cx<R> a, Cx<R> b) { return {a.r - b.r, a.i - b.i}; }
template <typename R> __device__ __forceinline__ Cx<R> operator*(Cx<R> a, Cx<R> b) {
    return {a.r * b.r - a.i * b.i, a.r * b.i + a.i * b.r};
}
template <typename R> __device__ __forceinline__ Cx<R> operator*(R s, Cx<R> a) { return {s * a.r, s * a.i}; }
template <typename R> __device__ __forceinline__ Cx<R> conj(Cx<R> a) { return {a.r, -a.i}; }
// a * conj(b)
template <typename R> __device__ __forceinline__ Cx<R> mul_conj(Cx<R> a, Cx<R> b) {
    return {a.r * b.r + a.i * b.i, a.i * b.r - a.r * b.i};
}
// conj(a) * b
template <typename R> __device__ __forceinline__ Cx<R> conj_mul(Cx<R> a, Cx<R> b) {
    return {a.r * b.r + a.i * b.i, a.r * b.i - a.i * b.r};
}
// i * a
template <typename R> __device__ __forceinline__ Cx<R> times_i(Cx<R> a) { return {-a.i, a.r}; }
template <typename R> __device__ __forceinline__ R norm2(Cx<R> a) { return a.r * a.r + a.i * a.i; }

// ---- fp32 complex arithmetic on the packed FP32x2 pipe (sm_100 FFMA2 / FADD2 / FMUL2).
// A complex number is one register pair: an add or a real scale is one instruction instead of
// two, and a complex multiply-accumulate two (scalar broadcast and pair-swap are operand
// modifiers of FFMA2) instead of four.  These overloads take precedence over the templates
// above for R = float; fp64 keeps the scalar forms.  Each lane rounds exactly as the scalar
// FADD/FMUL/FFMA would; only the contraction pattern of complex products differs from the
// compiler's scalar choice (within the fp32 / half parity tolerances).
__device__ __forceinline__ float2 f2(Cx<float> a) { return make_float2(a.r, a.i); }
__device__ __forceinline__ Cx<float> cf(float2 v) { return Cx<float>{v.x, v.y}; }
__device__ __forceinline__ float2 bc(float s) { return make_float2(s, s); }
__device__ __forceinline__ Cx<float> operator+(Cx<float> a, Cx<float> b) { return cf(__fadd2_rn(f2(a), f2(b))); }
__device__ __forceinline__ Cx<float> operator-(Cx<float> a, Cx<float> b) {
    return cf(__ffma2_rn(f2(b), bc(-1.f), f2(a)));
}
__device__ __forceinline__ Cx<float> operator*(float s, Cx<float> a) { return cf(__fmul2_rn(bc(s), f2(a))); }
// i a = (-a.i, a.r) and -i a = (a.i, -a.r) as FFMA2 operands: written as the FIRST operand with
// the scalar in the second, ptxas folds the pair swap and the one-lane negation into operand
// modifiers and the scalar into a broadcast — one FFMA2 per complex multiply-add term, exact
// (the sign change) and with no constant.  (The former i a = swap(a) * (-1, 1) needed that
// constant pair in registers, which ptxas rematerialised with two moves before most uses: +10 %
// instructions in the clover-inverse kernel, profiles/r02s_summary.md.)
__device__ __forceinline__ float2 i_pair(Cx<float> a) { return make_float2(-a.i, a.r); }
__device__ __forceinline__ float2 mi_pair(Cx<float> a) { return make_float2(a.i, -a.r); }
// acc + s * (i a), acc + s * (-i a)
__device__ __forceinline__ float2 fma_i(float2 acc, float s, Cx<float> a) { return __ffma2_rn(i_pair(a), bc(s), acc); }
__device__ __forceinline__ float2 fma_mi(float2 acc, float s, Cx<float> a) { return __ffma2_rn(mi_pair(a), bc(s), acc); }
__device__ __forceinline__ Cx<float> operator*(Cx<float> a, Cx<float> b) {
    return cf(fma_i(__fmul2_rn(bc(a.r), f2(b)), a.i, b));
}
__device__ __forceinline__ Cx<float> conj_mul(Cx<float> a, Cx<float> b) {
    return cf(fma_mi(__fmul2_rn(bc(a.r), f2(b)), a.i, b));
}

// p + S i q (S = +-1): one FFMA2 in fp32 (pair swap as operand modifier)
template <int S, typename R>
__device__ __forceinline__ Cx<R> add_i(Cx<R> p, Cx<R> q) {
    if constexpr (sizeof(R) == 4) {
        return cf(__fadd2_rn(f2(p), S > 0 ? i_pair(q) : mi_pair(q)));  // swap + one-lane negation: modifiers
    } else {
        return S > 0 ? Cx<R>{p.r - q.i, p.i + q.r} : Cx<R>{p.r + q.i, p.i - q.r};
    }
}
// acc + s g (real s)
template <typename R>
__device__ __forceinline__ Cx<R> axpy(R s, Cx<R> g, Cx<R> acc) {
    if constexpr (sizeof(R) == 4) return cf(__ffma2_rn(bc(s), f2(g), f2(acc)));
    else return acc + s * g;
}

// ----------------------------------------------------------------------------- precision traits
template <int P> struct Prec;
template <> struct Prec<8> { using R = double; };
template <> struct Prec<4> { using R = float; };
template <> struct Prec<2> { using R = float; };

constexpr float kHalfMax = 32767.0f;
constexpr float kHalfInv = 1.0f / 32767.0f;
// Half-precision spinor sites whose largest |component| is at most this are stored as zero
// (norm 0).  32767 / norm overflows fp32 below ~9.6e-35, and an infinite scale turns the
// zeros of such a site into NaN (0 * inf) in the requantised values the fused reductions use —
// seen deep in point-source solves, where the residual decays by > 30 orders of magnitude
// across the lattice.  The flushed values are < 1e-30 in absolute terms.
constexpr float kHalfTinyNorm = 1e-30f;

// cache-policy helpers: streamed data (links, clover) bypasses L1 allocation
__device__ __forceinline__ float4 ld_stream(const float4 *p) {
    float4 v;
    asm volatile("ld.global.nc.L1::no_allocate.v4.f32 {%0,%1,%2,%3}, [%4];"
                 : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w) : "l"(p));
    return v;
}
__device__ __forceinline__ double2 ld_stream(const double2 *p) {
    double2 v;
    asm volatile("ld.global.nc.L1::no_allocate.v2.f64 {%0,%1}, [%2];" : "=d"(v.x), "=d"(v.y) : "l"(p));
    return v;
}
__device__ __forceinline__ float2 ld_stream(const float2 *p) {
    float2 v;
    asm volatile("ld.global.nc.L1::no_allocate.v2.f32 {%0,%1}, [%2];" : "=f"(v.x), "=f"(v.y) : "l"(p));
    return v;
}
__device__ __forceinline__ short4 ld_stream(const short4 *p) {
    short4 v;
    asm volatile("ld.global.nc.L1::no_allocate.v4.s16 {%0,%1,%2,%3}, [%4];"
                 : "=h"(v.x), "=h"(v.y), "=h"(v.z), "=h"(v.w) : "l"(p));
    return v;
}
__device__ __forceinline__ short2 ld_stream(const short2 *p) {
    short2 v;
    asm volatile("ld.global.nc.L1::no_allocate.v2.s16 {%0,%1}, [%2];" : "=h"(v.x), "=h"(v.y) : "l"(p));
    return v;
}

// ----------------------------------------------------------------------------- SoA access
// Load reals [4*b0, 4*(b0+nb)) (fp32/half) or [2*b0, 2*(b0+nb)) (fp64) of site i.
// `stream` selects the no-L1-allocate path (links, clover) vs the read-only cached path.
// load modes: 0 = read-only path (L1-cached, non-coherent), 1 = streamed (no L1 allocation),
// 2 = L2 only (coherent with writes made by other CTAs earlier in the same kernel)
template <typename V> __device__ __forceinline__ V ld_mode2(const V *p) { return __ldcg(p); }
template <int P, int NB, int STREAM>
struct Blocks;

template <int NB, int STREAM>
struct Blocks<8, NB, STREAM> {
    static __device__ __forceinline__ void load(const void *base, long stride, long i, int b0, double *out) {
        const double2 *p = reinterpret_cast<const double2 *>(base);
#pragma unroll
        for (int k = 0; k < NB; ++k) {
            double2 v = STREAM == 1 ? ld_stream(p + (b0 + k) * stride + i)
                        : (STREAM == 2 ? __ldcg(p + (b0 + k) * stride + i) : __ldg(p + (b0 + k) * stride + i));
            out[2 * k] = v.x;
            out[2 * k + 1] = v.y;
        }
    }
    static __device__ __forceinline__ void store(void *base, long stride, long i, int b0, const double *in) {
        double2 *p = reinterpret_cast<double2 *>(base);
#pragma unroll
        for (int k = 0; k < NB; ++k) p[(b0 + k) * stride + i] = make_double2(in[2 * k], in[2 * k + 1]);
    }
};

template <int NB, int STREAM>
struct Blocks<4, NB, STREAM> {
    static __device__ __forceinline__ void load(const void *base, long stride, long i, int b0, float *out) {
        const float4 *p = reinterpret_cast<const float4 *>(base);
#pragma unroll
        for (int k = 0; k < NB; ++k) {
            float4 v = STREAM == 1 ? ld_stream(p + (b0 + k) * stride + i)
                       : (STREAM == 2 ? __ldcg(p + (b0 + k) * stride + i) : __ldg(p + (b0 + k) * stride + i));
            out[4 * k] = v.x;
            out[4 * k + 1] = v.y;
            out[4 * k + 2] = v.z;
            out[4 * k + 3] = v.w;
        }
    }
    static __device__ __forceinline__ void store(void *base, long stride, long i, int b0, const float *in) {
        float4 *p = reinterpret_cast<float4 *>(base);
#pragma unroll
        for (int k = 0; k < NB; ++k) p[(b0 + k) * stride + i] = make_float4(in[4 * k], in[4 * k + 1], in[4 * k + 2], in[4 * k + 3]);
    }
};

// ---- 16-bit fixed point <-> fp32 without the conversion (XU) pipe ------------------------
// The paper's half precision relied on the GT200 texture unit to turn int16 into floats
// (P:509-518).  On B200, I2F/F2I issue on the narrow XU pipe and become the limiter of the
// half-precision Dslash (ncu: XU 60% busy).  Both directions are exact fp32 integer tricks on
// the ALU/FMA pipes instead.  A quantised value q in [-32767, 32767] is stored OFFSET-BINARY,
// u = q + 32768 (the two's-complement bits with the sign bit flipped), so decoding is one
// byte-permute per value: bits(0x4B000000 | u) = 2^23 + u exactly, minus (2^23 + 2^15) = q.
//   float x (|x| <= 32767) -> RN-even u: low 16 bits of bits(x + 1.5*2^23 + 2^15).
constexpr uint32_t kHalfMagic = 0x4B000000u;
constexpr float kHalfBias = 8421376.0f;  // 2^23 + 2^15
__device__ __forceinline__ float i16lo_to_f32(uint32_t w) {
    return __uint_as_float(__byte_perm(w, kHalfMagic, 0x7610)) - kHalfBias;
}
__device__ __forceinline__ float i16hi_to_f32(uint32_t w) {
    return __uint_as_float(__byte_perm(w, kHalfMagic, 0x7632)) - kHalfBias;
}
// both values of a stored word, times `scale`: 2 PRMT + FADD2 + FMUL2 (same rounding as the
// scalar FADD then FMUL)
__device__ __forceinline__ float2 dq2(uint32_t w, float scale) {
    const float2 b = make_float2(__uint_as_float(__byte_perm(w, kHalfMagic, 0x7610)),
                                 __uint_as_float(__byte_perm(w, kHalfMagic, 0x7632)));
    return __fmul2_rn(bc(scale), __fadd2_rn(b, bc(-kHalfBias)));
}
// both values of a stored word as the integers they hold (no scale): 2 PRMT + FADD2.  The
// deferred-scale half Dslash multiplies the per-site scale into the accumulation instead.
__device__ __forceinline__ float2 dq2_q(uint32_t w) {
    const float2 b = make_float2(__uint_as_float(__byte_perm(w, kHalfMagic, 0x7610)),
                                 __uint_as_float(__byte_perm(w, kHalfMagic, 0x7632)));
    return __fadd2_rn(b, bc(-kHalfBias));
}
// a * inv, b * inv -> packed offset-binary pair: one FFMA2 rounds each exact product to the
// nearest integer (even on ties) — one rounding, no intermediate fp32 product
__device__ __forceinline__ uint32_t f32x2_scale_to_i16x2(float a, float b, float inv) {
    const float2 r = __ffma2_rn(make_float2(a, b), bc(inv), bc(12615680.0f));  // 1.5*2^23 + 2^15
    return __byte_perm(__float_as_uint(r.x), __float_as_uint(r.y), 0x5410);
}
// the integer round(x * inv) (exactly what f32x2_scale_to_i16x2 stores), as a float
__device__ __forceinline__ float q_scaled_as_f32(float x, float inv) {
    return __fmaf_rn(x, inv, 12582912.0f) - 12582912.0f;
}
// host/device: quantised integer q -> stored 16-bit word
__host__ __device__ __forceinline__ short h16_code(int q) { return (short)(uint16_t)((unsigned)q ^ 0x8000u); }
__device__ __forceinline__ uint2 ld_stream_u2(const uint2 *p) {
    uint2 v;
    asm volatile("ld.global.nc.L1::no_allocate.v2.u32 {%0,%1}, [%2];" : "=r"(v.x), "=r"(v.y) : "l"(p));
    return v;
}


// ---- half storage records.  Every 16-bit field is stored in 16-byte words first: a 12-real
// record (half spinor, face, recon-12 link) is one uint4 (reals 0-7) + one uint2 (reals 8-11),
// each in its own site-major region, so a warp load moves 512 B per instruction (an 8-byte
// layout needs twice the load instructions and outstanding requests per byte).
__device__ __forceinline__ uint4 ld_stream_u4(const uint4 *p) {
    uint4 v;
    asm volatile("ld.global.nc.L1::no_allocate.v4.u32 {%0,%1,%2,%3}, [%4];"
                 : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "l"(p));
    return v;
}
// MODE 0: read-only path; 1: streamed (no L1 allocation); 2: L2 only (coherent)
template <int MODE, typename V>
__device__ __forceinline__ V ld_m(const V *p) {
    if constexpr (MODE == 2) return __ldcg(p);
    else if constexpr (MODE == 1) {
        if constexpr (std::is_same<V, uint4>::value) return ld_stream_u4(p);
        else if constexpr (std::is_same<V, uint2>::value) return ld_stream_u2(p);
        else return __ldg(p);
    } else return __ldg(p);
}
struct H12 {
    uint4 u;
    uint2 v;
    template <int MODE>
    __device__ __forceinline__ void load(const void *ureg, const void *vreg, long i) {
        u = ld_m<MODE>(reinterpret_cast<const uint4 *>(ureg) + i);
        v = ld_m<MODE>(reinterpret_cast<const uint2 *>(vreg) + i);
    }
    __device__ __forceinline__ void decode(float scale, float *out) const {
        const uint32_t w[6] = {u.x, u.y, u.z, u.w, v.x, v.y};
#pragma unroll
        for (int k = 0; k < 6; ++k) {
            const float2 d = dq2(w[k], scale);
            out[2 * k] = d.x;
            out[2 * k + 1] = d.y;
        }
    }
    __device__ __forceinline__ void decode_q(float *out) const {
        const uint32_t w[6] = {u.x, u.y, u.z, u.w, v.x, v.y};
#pragma unroll
        for (int k = 0; k < 6; ++k) {
            const float2 d = dq2_q(w[k]);
            out[2 * k] = d.x;
            out[2 * k + 1] = d.y;
        }
    }
    __device__ __forceinline__ void encode(const float *in, float inv) {
        uint32_t w[6];
#pragma unroll
        for (int k = 0; k < 6; ++k) w[k] = f32x2_scale_to_i16x2(in[2 * k], in[2 * k + 1], inv);
        u = make_uint4(w[0], w[1], w[2], w[3]);
        v = make_uint2(w[4], w[5]);
    }
    __device__ __forceinline__ void store(void *ureg, void *vreg, long i) const {
        reinterpret_cast<uint4 *>(ureg)[i] = u;
        reinterpret_cast<uint2 *>(vreg)[i] = v;
    }
};
// region addresses.  Half spinor field: [U upper][U lower][V upper][V lower][norm] x stride;
// face: [U][V][norm] x fstride.
__device__ __forceinline__ const char *cptr(const void *b, size_t off) { return reinterpret_cast<const char *>(b) + off; }
__device__ __forceinline__ char *mptr(void *b, size_t off) { return reinterpret_cast<char *>(b) + off; }
__device__ __forceinline__ size_t h_spinor_u(long stride, int hf) { return (size_t)16 * stride * hf; }
__device__ __forceinline__ size_t h_spinor_v(long stride, int hf) { return (size_t)(32 + 8 * hf) * stride; }

// ----------------------------------------------------------------------------- spinors
// A spinor field: 24 reals per site (spin-major, colour, re/im) in the NR basis.
// fp64: 12 double2 blocks; fp32: 6 float4 blocks; half: two H12 records (upper spins 0,1 and
// lower spins 2,3) + float norm[stride].
template <int P>
struct SpinorIO {
    using R = typename Prec<P>::R;
    static constexpr int BPH = (P == 8) ? 6 : 3;  // blocks per 12-real half-spinor

    // norm array (half only) follows the 48 bytes x stride of the four half regions
    static __device__ __forceinline__ const float *norms(const void *base, long stride) {
        return reinterpret_cast<const float *>(reinterpret_cast<const char *>(base) + (size_t)6 * 8 * stride);
    }
    static __device__ __forceinline__ float *norms(void *base, long stride) {
        return reinterpret_cast<float *>(reinterpret_cast<char *>(base) + (size_t)6 * 8 * stride);
    }

    // half = 0: reals 0..11 (spins 0,1), half = 1: reals 12..23 (spins 2,3)
    // MODE 0: read-only path; MODE 2: L2-coherent (data written earlier in the same kernel)
    template <int MODE = 0>
    static __device__ __forceinline__ void load_half(const void *base, long stride, long i, int half, R *out) {
        if constexpr (P == 2) {
            const float nrm = ld_m<MODE>(norms(base, stride) + i);
            H12 r;
            r.load<MODE>(cptr(base, h_spinor_u(stride, half)), cptr(base, h_spinor_v(stride, half)), i);
            r.decode(nrm * kHalfInv, out);
        } else {
            Blocks<P, BPH, MODE>::load(base, stride, i, BPH * half, out);
        }
    }
    template <int MODE = 0>
    static __device__ __forceinline__ void load(const void *base, long stride, long i, R *out) {
        load_half<MODE>(base, stride, i, 0, out);
        load_half<MODE>(base, stride, i, 1, out + 12);
    }
    static __device__ __forceinline__ void store(void *base, long stride, long i, const R *in) {
        if constexpr (P == 2) {
            float m = 0.f;
#pragma unroll
            for (int k = 0; k < 24; ++k) m = fmaxf(m, fabsf(in[k]));
            if (m <= kHalfTinyNorm) m = 0.f;  // flush (a NaN norm stays NaN: breakdown detection)
            norms(base, stride)[i] = m;
            const float inv = (m > 0.f) ? kHalfMax / m : 0.f;
#pragma unroll
            for (int hf = 0; hf < 2; ++hf) {
                H12 r;
                r.encode(in + 12 * hf, inv);
                r.store(mptr(base, h_spinor_u(stride, hf)), mptr(base, h_spinor_v(stride, hf)), i);
            }
        } else {
            Blocks<P, 2 * BPH, false>::store(base, stride, i, 0, in);
        }
    }
    // store, and replace `v` by exactly what a later load() of this site returns (half:
    // the dequantised values) — lets a kernel reduce over what it stored without re-reading
    // its own output through the non-coherent read-only path.
    static __device__ __forceinline__ void store_requant(void *base, long stride, long i, R *v) {
        store(base, stride, i, v);
        if constexpr (P == 2) {
            float m = 0.f;
#pragma unroll
            for (int k = 0; k < 24; ++k) m = fmaxf(m, fabsf(v[k]));
            if (m <= kHalfTinyNorm) m = 0.f;
            const float inv = (m > 0.f) ? kHalfMax / m : 0.f;
            const float scale = m * kHalfInv;
#pragma unroll
            for (int k = 0; k < 24; ++k) v[k] = __fmul_rn(scale, q_scaled_as_f32(v[k], inv));
        }
    }
};

// A face (12 reals per site): fp64 6 double2, fp32 3 float4, half one H12 + float norm[fstride]
template <int P>
struct FaceIO {
    using R = typename Prec<P>::R;
    static constexpr int NB = (P == 8) ? 6 : 3;
    static __device__ __forceinline__ const float *norms(const void *base, long fs) {
        return reinterpret_cast<const float *>(reinterpret_cast<const char *>(base) + (size_t)3 * 8 * fs);
    }
    static __device__ __forceinline__ float *norms(void *base, long fs) {
        return reinterpret_cast<float *>(reinterpret_cast<char *>(base) + (size_t)3 * 8 * fs);
    }
    static __device__ __forceinline__ void load(const void *base, long fs, long f, R *out) {
        if constexpr (P == 2) {
            const float nrm = __ldg(norms(base, fs) + f);
            H12 r;
            r.load<0>(base, cptr(base, (size_t)16 * fs), f);
            r.decode(nrm * kHalfInv, out);
        } else {
            Blocks<P, NB, false>::load(base, fs, f, 0, out);
        }
    }
};

// Half links: RECON/8 uint4 regions, then a uint2 region (RECON % 8 == 4), then a uint32
// region (RECON % 4 == 2) — recon-12: 16 + 8 B, recon-18: 16 + 16 + 4 B, recon-8: 16 B.
template <int RECON>
struct HLink {
    static constexpr int N16 = RECON / 8;
    static constexpr bool kV = (RECON % 8) >= 4;
    static constexpr bool kW = (RECON % 4) == 2;
    uint4 u[N16];
    uint2 v;
    uint32_t w;
    __device__ __forceinline__ void load(const void *base, long stride, long i) {
#pragma unroll
        for (int k = 0; k < N16; ++k) u[k] = ld_stream_u4(reinterpret_cast<const uint4 *>(cptr(base, (size_t)16 * k * stride)) + i);
        size_t off = (size_t)16 * N16 * stride;
        if constexpr (kV) {
            v = ld_stream_u2(reinterpret_cast<const uint2 *>(cptr(base, off)) + i);
            off += (size_t)8 * stride;
        }
        if constexpr (kW) w = __ldg(reinterpret_cast<const uint32_t *>(cptr(base, off)) + i);
    }
    __device__ __forceinline__ void decode(float *raw) const {
#pragma unroll
        for (int k = 0; k < N16; ++k) {
            const uint32_t q[4] = {u[k].x, u[k].y, u[k].z, u[k].w};
#pragma unroll
            for (int j = 0; j < 4; ++j) {
                const float2 d = dq2(q[j], kHalfInv);
                raw[8 * k + 2 * j] = d.x;
                raw[8 * k + 2 * j + 1] = d.y;
            }
        }
        if constexpr (kV) {
            const float2 a = dq2(v.x, kHalfInv), b = dq2(v.y, kHalfInv);
            raw[8 * N16] = a.x; raw[8 * N16 + 1] = a.y; raw[8 * N16 + 2] = b.x; raw[8 * N16 + 3] = b.y;
        }
        if constexpr (kW) {
            const float2 a = dq2(w, kHalfInv);
            raw[RECON - 2] = a.x;
            raw[RECON - 1] = a.y;
        }
    }
    // the stored integers (link = kHalfInv * raw)
    __device__ __forceinline__ void decode_q(float *raw) const {
#pragma unroll
        for (int k = 0; k < N16; ++k) {
            const uint32_t q[4] = {u[k].x, u[k].y, u[k].z, u[k].w};
#pragma unroll
            for (int j = 0; j < 4; ++j) {
                const float2 d = dq2_q(q[j]);
                raw[8 * k + 2 * j] = d.x;
                raw[8 * k + 2 * j + 1] = d.y;
            }
        }
        if constexpr (kV) {
            const float2 a = dq2_q(v.x), b = dq2_q(v.y);
            raw[8 * N16] = a.x; raw[8 * N16 + 1] = a.y; raw[8 * N16 + 2] = b.x; raw[8 * N16 + 3] = b.y;
        }
        if constexpr (kW) {
            const float2 a = dq2_q(w);
            raw[RECON - 2] = a.x;
            raw[RECON - 1] = a.y;
        }
    }
};

// ----------------------------------------------------------------------------- links
// Stored reals per link: 18: u[r][c] (re,im); 12: rows 0,1; 8: (theta0, theta2, u01, u02, u10)
// with theta0 = arg u00, theta2 = arg u20 (half: theta/pi).  Reconstruction in registers:
// two-row: row2 = conj(row0 x row1); eight-parameter: reading Q6.
template <int P, int RECON>
struct LinkIO {
    using R = typename Prec<P>::R;
    static __device__ __forceinline__ void load_raw(const void *base, long stride, long i, R *raw) {
        if constexpr (P == 2) {
            HLink<RECON> h;
            h.load(base, stride, i);
            h.decode(raw);
        } else {
            constexpr int NB4 = (P == 8) ? RECON / 2 : RECON / 4;
            Blocks<P, NB4, true>::load(base, stride, i, 0, raw);
            if constexpr (P == 4 && (RECON % 4) != 0) {  // trailing 2-real block (recon 18)
                const float2 *p2 = reinterpret_cast<const float2 *>(reinterpret_cast<const char *>(base) +
                                                                    (size_t)NB4 * 16 * stride);
                float2 v = ld_stream(p2 + i);
                raw[RECON - 2] = v.x;
                raw[RECON - 1] = v.y;
            }
        }
    }

    // full 3x3 link u[row][col]
    static __device__ __forceinline__ void load(const void *base, long stride, long i, Cx<R> u[3][3]) {
        R raw[RECON];
        load_raw(base, stride, i, raw);
        reconstruct(raw, u);
    }
    static __device__ __forceinline__ void reconstruct(const R *raw, Cx<R> u[3][3]) {
        if constexpr (RECON == 18) {
#pragma unroll
            for (int r = 0; r < 3; ++r)
#pragma unroll
                for (int c = 0; c < 3; ++c) u[r][c] = cx(raw[(r * 3 + c) * 2], raw[(r * 3 + c) * 2 + 1]);
        } else if constexpr (RECON == 12) {
#pragma unroll
            for (int r = 0; r < 2; ++r)
#pragma unroll
                for (int c = 0; c < 3; ++c) u[r][c] = cx(raw[(r * 3 + c) * 2], raw[(r * 3 + c) * 2 + 1]);
            // row2 = conj(row0 x row1).  Half precision (QX_XREC bit 0; bit 1 fp32, measured
            // slower there): with conj(row 1) formed once, 4 FMUL2/FFMA2 per element (scalar
            // broadcast / negation and the pair swap are operand modifiers) instead of two
            // complex products, a subtraction and a conjugation (h-12 inverse-xpay -2 %)
#ifndef QX_XREC
#define QX_XREC 1
#endif
#if QX_XREC
            if constexpr (sizeof(R) == 4 && (QX_XREC >> (P == 2 ? 0 : 1) & 1)) {
                // conj(x y - z w) = x.r conj(y) - x.i swap(y) - z.r conj(w) + z.i swap(w); the
                // conjugations, swaps and negations are operand modifiers of the first (pair)
                // operand, the scalars broadcasts of the second — no constant pair
                auto cross = [&](int xa, int yb, int za, int wb) {
                    const Cx<float> xx = u[0][xa], zz = u[0][za], y = u[1][yb], w = u[1][wb];
                    float2 r = __fmul2_rn(make_float2(y.r, -y.i), bc(xx.r));
                    r = __ffma2_rn(make_float2(-y.i, -y.r), bc(xx.i), r);
                    r = __ffma2_rn(make_float2(-w.r, w.i), bc(zz.r), r);
                    return cf(__ffma2_rn(make_float2(w.i, w.r), bc(zz.i), r));
                };
                const Cx<float> a0 = cross(1, 2, 2, 1), a1 = cross(2, 0, 0, 2), a2 = cross(0, 1, 1, 0);
                u[2][0] = a0; u[2][1] = a1; u[2][2] = a2;
                return;
            }
#endif
            u[2][0] = conj(u[0][1] * u[1][2] - u[0][2] * u[1][1]);
            u[2][1] = conj(u[0][2] * u[1][0] - u[0][0] * u[1][2]);
            u[2][2] = conj(u[0][0] * u[1][1] - u[0][1] * u[1][0]);
        } else {
            R th0 = raw[0], th2 = raw[1];
            if constexpr (P == 2) {
                th0 *= (R)3.14159265358979323846;
                th2 *= (R)3.14159265358979323846;
            }
            Cx<R> u01 = cx(raw[2], raw[3]), u02 = cx(raw[4], raw[5]), u10 = cx(raw[6], raw[7]);
            R n = norm2(u01) + norm2(u02);
            R a00 = sqrt_(fmax((R)0, (R)1 - n));
            R s0, c0, s2, c2;
            sincos_(th0, &s0, &c0);
            sincos_(th2, &s2, &c2);
            Cx<R> u00 = cx(a00 * c0, a00 * s0);
            R a20 = sqrt_(fmax((R)0, (R)1 - a00 * a00 - norm2(u10)));
            Cx<R> u20 = cx(a20 * c2, a20 * s2);
            R inv = rcp_(n);
            Cx<R> A = conj_mul(u00, u10);
            Cx<R> C = conj_mul(u00, u20);
            Cx<R> cu20 = conj(u20), cu10 = conj(u10), cu01 = conj(u01), cu02 = conj(u02);
            u[0][0] = u00; u[0][1] = u01; u[0][2] = u02;
            u[1][0] = u10;
            u[2][0] = u20;
            u[1][1] = (-inv) * (cu20 * cu02 + A * u01);
            u[1][2] = inv * (cu20 * cu01 - A * u02);
            u[2][1] = inv * (cu10 * cu02 - C * u01);
            u[2][2] = (-inv) * (cu10 * cu01 + C * u02);
        }
    }

    // fp64: accurate; fp32/half: SFU approximations (abs error ~4e-7 on [-pi, pi], far inside
    // the 1e-5 / 5e-3 budgets) — the accurate fp32 versions made recon-8 instruction-bound
    static __device__ __forceinline__ void sincos_(double x, double *s, double *c) { sincos(x, s, c); }
    static __device__ __forceinline__ void sincos_(float x, float *s, float *c) { __sincosf(x, s, c); }
    static __device__ __forceinline__ double sqrt_(double x) { return sqrt(x); }
    static __device__ __forceinline__ float sqrt_(float x) { return x * rsqrtf(fmaxf(x, 1e-30f)); }
    static __device__ __forceinline__ double rcp_(double x) { return 1.0 / x; }
    static __device__ __forceinline__ float rcp_(float x) { return __fdividef(1.0f, x); }
};

// ----------------------------------------------------------------------------- raw site data
// Undecoded loads, so the Dslash can issue the loads of two hops before consuming either
// (half: the 16-bit words + norm stay packed, half the registers of the decoded values).
template <int P> struct StoreVec;
template <> struct StoreVec<8> { using V = double2; };
template <> struct StoreVec<4> { using V = float4; };
template <> struct StoreVec<2> { using V = uint4; };

// NREAL = 24 (spinor) or 12 (half spinor / face)
template <int P, int NREAL>
struct RawVec {
    using R = typename Prec<P>::R;
    static constexpr int RPV = (P == 8) ? 2 : 4;   // reals per stored vector (fp64 / fp32)
    static constexpr int NB = NREAL / RPV;
    typename StoreVec<P == 2 ? 4 : P>::V d[P == 2 ? 1 : NB];  // fp64 / fp32 blocks
    H12 h[NREAL / 12];                                       // half records
    float n;                                                 // half: the site norm
    template <int MODE>
    __device__ __forceinline__ void load_blocks(const void *base, long stride, long i, int b0) {
        using V = typename StoreVec<P>::V;
        const V *p = reinterpret_cast<const V *>(base);
#pragma unroll
        for (int k = 0; k < NB; ++k) d[k] = ld_m<MODE>(p + (b0 + k) * stride + i);
    }
    template <int MODE>
    __device__ __forceinline__ void load_spinor(const void *base, long stride, long i) {
        if constexpr (P == 2) {
#pragma unroll
            for (int hf = 0; hf < 2; ++hf)
                h[hf].template load<MODE>(cptr(base, h_spinor_u(stride, hf)), cptr(base, h_spinor_v(stride, hf)), i);
            n = ld_m<MODE>(SpinorIO<2>::norms(base, stride) + i);
        } else {
            load_blocks<MODE>(base, stride, i, 0);
        }
    }
    template <int MODE>
    __device__ __forceinline__ void load_half(const void *base, long stride, long i, int hf) {
        if constexpr (P == 2) {
            h[0].template load<MODE>(cptr(base, h_spinor_u(stride, hf)), cptr(base, h_spinor_v(stride, hf)), i);
            n = ld_m<MODE>(SpinorIO<2>::norms(base, stride) + i);
        } else {
            load_blocks<MODE>(base, stride, i, NB * hf);
        }
    }
    __device__ __forceinline__ void load_face(const void *base, long fs, long f) {
        if constexpr (P == 2) {
            h[0].template load<0>(base, cptr(base, (size_t)16 * fs), f);
            n = __ldg(FaceIO<2>::norms(base, fs) + f);
        } else {
            load_blocks<0>(base, fs, f, 0);
        }
    }
    // identical values to SpinorIO / FaceIO loads
    __device__ __forceinline__ void decode(R *out) const {
        if constexpr (P == 8) {
#pragma unroll
            for (int k = 0; k < NB; ++k) {
                out[2 * k] = d[k].x;
                out[2 * k + 1] = d[k].y;
            }
        } else if constexpr (P == 4) {
#pragma unroll
            for (int k = 0; k < NB; ++k) {
                out[4 * k] = d[k].x; out[4 * k + 1] = d[k].y; out[4 * k + 2] = d[k].z; out[4 * k + 3] = d[k].w;
            }
        } else {
            const float scale = n * kHalfInv;
#pragma unroll
            for (int r = 0; r < NREAL / 12; ++r) h[r].decode(scale, out + 12 * r);
        }
    }
    // half: the stored integers plus the bias kHalfBias = 2^23 + 2^15, as fp32 (one PRMT per
    // value, no arithmetic): the spatial projection removes the bias exactly (dslash.cuh)
    __device__ __forceinline__ void decode_b(float *out) const {
#pragma unroll
        for (int r = 0; r < NREAL / 12; ++r) {
            const uint32_t w[6] = {h[r].u.x, h[r].u.y, h[r].u.z, h[r].u.w, h[r].v.x, h[r].v.y};
#pragma unroll
            for (int k = 0; k < 6; ++k) {
                out[12 * r + 2 * k] = __uint_as_float(__byte_perm(w[k], kHalfMagic, 0x7610));
                out[12 * r + 2 * k + 1] = __uint_as_float(__byte_perm(w[k], kHalfMagic, 0x7632));
            }
        }
    }
    // half: the stored integers; value = scale() * out
    __device__ __forceinline__ void decode_q(float *out) const {
#pragma unroll
        for (int r = 0; r < NREAL / 12; ++r) h[r].decode_q(out + 12 * r);
    }
    __device__ __forceinline__ float scale() const { return n * kHalfInv; }
};

template <int P, int RECON>
struct RawLink {
    using R = typename Prec<P>::R;
    static constexpr int NB = (P == 8) ? RECON / 2 : RECON / 4;
    static constexpr bool kTail = (P == 4) && (RECON % 4) != 0;
    typename StoreVec<P == 2 ? 4 : P>::V d[P == 2 ? 1 : NB];
    float2 tail;
    HLink<RECON> h;
    __device__ __forceinline__ void load(const void *base, long stride, long i) {
        if constexpr (P == 2) {
            h.load(base, stride, i);
        } else {
            using V = typename StoreVec<P>::V;
            const V *p = reinterpret_cast<const V *>(base);
#pragma unroll
            for (int k = 0; k < NB; ++k) d[k] = ld_stream(p + k * stride + i);
            if constexpr (kTail)
                tail = ld_stream(reinterpret_cast<const float2 *>(cptr(base, (size_t)NB * sizeof(V) * stride)) + i);
        }
    }
    // identical to LinkIO<P, RECON>::load
    __device__ __forceinline__ void decode(Cx<R> u[3][3]) const {
        R raw[RECON];
        if constexpr (P == 8) {
#pragma unroll
            for (int k = 0; k < NB; ++k) {
                raw[2 * k] = d[k].x;
                raw[2 * k + 1] = d[k].y;
            }
        } else if constexpr (P == 4) {
#pragma unroll
            for (int k = 0; k < NB; ++k) {
                raw[4 * k] = d[k].x; raw[4 * k + 1] = d[k].y; raw[4 * k + 2] = d[k].z; raw[4 * k + 3] = d[k].w;
            }
            if constexpr (kTail) {
                raw[RECON - 2] = tail.x;
                raw[RECON - 1] = tail.y;
            }
        } else {
            h.decode(raw);
        }
        LinkIO<P, RECON>::reconstruct(raw, u);
    }
    // half, recon 18/12: the link in units of kHalfInv (the stored integers; the two-row
    // reconstruction's third row, quadratic in them, is brought back to the same units)
    __device__ __forceinline__ void decode_q(Cx<R> u[3][3]) const {
        static_assert(P == 2 && RECON != 8, "deferred-scale decode: half recon 18/12 only");
        R raw[RECON];
        h.decode_q(raw);
        LinkIO<P, RECON>::reconstruct(raw, u);
        if constexpr (RECON == 12) {
#pragma unroll
            for (int c = 0; c < 3; ++c) u[2][c] = kHalfInv * u[2][c];
        }
    }
};

}  // namespace qx

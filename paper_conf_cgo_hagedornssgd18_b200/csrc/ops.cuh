// ops.cuh — the neighbourhood functions f of map.
//
// Every kernel family (K0 generic, K1 2D tile, K2 3D sweep) evaluates f
// through these functions, so each output point sees exactly the same fp32
// operation sequence whatever kernel, tile shape or GPU count produced it
// (tiling independence; A12).  The library is compiled
// with -fmad=false: the only fused multiply-adds are the explicit __fmaf_rn
// below, so the compiler cannot contract differently in different kernels.
//
// An accessor ``W`` exposes the window: ``W.template at<DZ, DY, DX>()`` is
// the padded input at offset (DZ, DY, DX) from the window centre (for the
// centred ops below); point-wise zipped inputs are passed as values.
#pragma once
#include <type_traits>
#include <utility>

#include "common.cuh"

namespace lift {

// ---- scalar and packed arithmetic -----------------------------------------
// The map functions below are written once over a value type V: float (one
// output) or float2 (two outputs in the two fp32 lanes of sm_100a's packed
// FFMA2 / FADD2 / FMUL2 — half the instructions for issue-bound kernels).
// Each packed lane is the same IEEE round-to-nearest operation as the scalar
// one, so an output's bits do not depend on which form computed it.
__device__ __forceinline__ float vfma(float a, float b, float c) { return __fmaf_rn(a, b, c); }
__device__ __forceinline__ float vadd(float a, float b) { return __fadd_rn(a, b); }
__device__ __forceinline__ float vsub(float a, float b) { return __fsub_rn(a, b); }
__device__ __forceinline__ float vmul(float a, float b) { return __fmul_rn(a, b); }
__device__ __forceinline__ float2 vfma(float2 a, float2 b, float2 c) { return __ffma2_rn(a, b, c); }
__device__ __forceinline__ float2 vadd(float2 a, float2 b) { return __fadd2_rn(a, b); }
__device__ __forceinline__ float2 vmul(float2 a, float2 b) { return __fmul2_rn(a, b); }
__device__ __forceinline__ float2 vsub(float2 a, float2 b) {
  unsigned long long r;
  asm("sub.rn.f32x2 %0, %1, %2;"
      : "=l"(r)
      : "l"(*reinterpret_cast<const unsigned long long*>(&a)), "l"(*reinterpret_cast<const unsigned long long*>(&b)));
  return *reinterpret_cast<float2*>(&r);
}
template <class V>
__device__ __forceinline__ V vbc(float s);
template <>
__device__ __forceinline__ float vbc<float>(float s) { return s; }
template <>
__device__ __forceinline__ float2 vbc<float2>(float s) { return make_float2(s, s); }

template <class Acc>
using acc_value_t = std::decay_t<decltype(std::declval<const Acc&>().template at<0, 0, 0>())>;

// compile-time loop: f(std::integral_constant<int, 0..N-1>) in order
template <class F, int... Is>
__device__ __forceinline__ void static_for_impl(F&& f, std::integer_sequence<int, Is...>) {
  (f(std::integral_constant<int, Is>{}), ...);
}
template <int N, class F>
__device__ __forceinline__ void static_for(F&& f) {
  static_for_impl(f, std::make_integer_sequence<int, N>{});
}

// ---- WEIGHTED: sum_k w_k * W[k] over a centred (2RZ+1)x(2RY+1)x(2RX+1) window,
// taps in row-major window order (the order K0 uses for its non-zero taps;
// a zero-weight tap is an exact no-op: fma(0, x, acc) == acc for finite x).
// STAR restricts the taps to the axes (7/13-point Jacobi); otherwise the box.
template <int RZ, int RY, int RX, bool STAR, class Acc>
__device__ __forceinline__ float op_weighted(const Acc& W, const float* wbox) {
  constexpr int SZ = 2 * RZ + 1, SY = 2 * RY + 1, SX = 2 * RX + 1;
  float acc = 0.0f;
  static_for<SZ * SY * SX>([&](auto K) {
    constexpr int k = decltype(K)::value;
    constexpr int kz = k / (SY * SX), ky = (k / SX) % SY, kx = k % SX;
    constexpr int nax = (kz != RZ) + (ky != RY) + (kx != RX);
    if constexpr (!STAR || nax <= 1) acc = __fmaf_rn(wbox[k], W.template at<kz - RZ, ky - RY, kx - RX>(), acc);
  });
  return acc;
}

// ---- Hotspot3D (Rodinia v3.1 hotspot3D; A16) ---------------------
// T' = cc*C + cn*N + cs*S + ce*E + cw*W + ct*T + cb*B + sdc*P + ct*amb
// N = y-1, S = y+1, W = x-1, E = x+1, B = z-1, T = z+1.
template <class Acc>
__device__ __forceinline__ float op_hotspot3d(const Acc& T, float Pc, const float* prm) {
  const float cc = prm[0], cn = prm[1], cs = prm[2], ce = prm[3], cw = prm[4];
  const float ct = prm[5], cb = prm[6], sdc = prm[7], amb = prm[8];
  float acc = __fmul_rn(cc, T.template at<0, 0, 0>());
  acc = __fmaf_rn(cn, T.template at<0, -1, 0>(), acc);
  acc = __fmaf_rn(cs, T.template at<0, 1, 0>(), acc);
  acc = __fmaf_rn(ce, T.template at<0, 0, 1>(), acc);
  acc = __fmaf_rn(cw, T.template at<0, 0, -1>(), acc);
  acc = __fmaf_rn(ct, T.template at<1, 0, 0>(), acc);
  acc = __fmaf_rn(cb, T.template at<-1, 0, 0>(), acc);
  acc = __fmaf_rn(sdc, Pc, acc);
  acc = __fmaf_rn(ct, amb, acc);
  return acc;
}

// Reciprocal and reciprocal square root: the SFU approximation (MUFU, rel.
// error ~2^-23) refined by one Newton step in explicit FMAs.  Branch-free
// (the correctly rounded __frcp_rn / __frsqrt_rn carry a range check and a
// slow path: ~10 instructions and a branch per point); within 2 ulp of the
// exact value for normal inputs — far inside the 1e-5 parity bound — and
// identical in every kernel family (reading A24b).
__device__ __forceinline__ float rcp_approx(float x) {
  float r;
  asm("rcp.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(x));
  return r;
}
__device__ __forceinline__ float rcp_nr(float x) {
  const float r = rcp_approx(x);
  const float e = __fmaf_rn(-x, r, 1.0f);
  return __fmaf_rn(r, e, r);
}
// two lanes: the same MUFU approximation per lane, the same Newton step packed
__device__ __forceinline__ float2 rcp_nr(float2 x) {
  const float2 r = make_float2(rcp_approx(x.x), rcp_approx(x.y));
  const float2 e = vfma(make_float2(-x.x, -x.y), r, vbc<float2>(1.0f));
  return vfma(r, e, r);
}
// c clamped to [0, 1]; a NaN stays NaN (as the select form c < 0 ? 0 :
// (c > 1 ? 1 : c) does): max.NaN / min.NaN, two FMNMX instead of a
// compare-select chain
__device__ __forceinline__ float clamp01(float c) {
  float r;
  asm("max.NaN.f32 %0, %1, 0f00000000;" : "=f"(r) : "f"(c));
  asm("min.NaN.f32 %0, %0, 0f3F800000;" : "+f"(r));
  return r;
}
__device__ __forceinline__ float2 clamp01(float2 c) { return make_float2(clamp01(c.x), clamp01(c.y)); }
__device__ __forceinline__ float rsqrt_nr(float x) {
  float r;
  asm("rsqrt.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(x));
  // r' = r + r/2 * (1 - x r^2)
  const float e = __fmaf_rn(-x, __fmul_rn(r, r), 1.0f);
  return __fmaf_rn(__fmul_rn(0.5f, r), e, r);
}

// ---- SRAD kernel 1: I -> c (Rodinia v3.1 srad; A18) --------------
// Definition: G2 = g/Ic^2, L = sd/Ic (g = sum dX^2, sd = sum dX),
// q = (G2/2 - L^2/16) / (1 + L/4)^2, d = (q - q0)/(q0(1+q0)), c = 1/(1+d).
// Multiplying through by Ic^2 gives the same function with one reciprocal and
// only non-negative terms (reading A18b):
//   D = Ic + sd/4,  n0 = g/2 - sd^2/16 (>= g/4 by Cauchy-Schwarz),
//   c = D^2 / (a*D^2 + b*n0),  a = q0/(1+q0),  b = 1/(q0(1+q0))
// with a, b plan constants (prm[1], prm[2]); then c is clamped to [0, 1].
template <class Acc>
__device__ __forceinline__ acc_value_t<Acc> op_srad1(const Acc& I, const float* prm) {
  using V = acc_value_t<Acc>;
  const V a = vbc<V>(prm[1]), b = vbc<V>(prm[2]);
  const V Ic = I.template at<0, 0, 0>();
  const V dN = vsub(I.template at<0, -1, 0>(), Ic);
  const V dS = vsub(I.template at<0, 1, 0>(), Ic);
  const V dW = vsub(I.template at<0, 0, -1>(), Ic);
  const V dE = vsub(I.template at<0, 0, 1>(), Ic);
  V g = vmul(dN, dN);
  g = vfma(dS, dS, g);
  g = vfma(dW, dW, g);
  g = vfma(dE, dE, g);
  const V sd = vadd(vadd(vadd(dN, dS), dW), dE);
  const V n0 = vfma(vbc<V>(-0.0625f), vmul(sd, sd), vmul(vbc<V>(0.5f), g));
  const V D = vfma(vbc<V>(0.25f), sd, Ic);
  const V D2 = vmul(D, D);
  const V c = vmul(D2, rcp_nr(vfma(a, D2, vmul(b, n0))));
  return clamp01(c);
}

// SRAD1's constants {q0, a, b} from q0 (the same derivation as the plan's)
__host__ __device__ inline void srad1_constants(float q0f, float* out3) {
  const double q0 = q0f;
  out3[0] = q0f;
  out3[1] = (float)(q0 / (1.0 + q0));
  out3[2] = (float)(1.0 / (q0 * (1.0 + q0)));
}

// q0^2 = var(I) / mean(I)^2 from fp64 (sum, sum of squares) over n points
// (Rodinia SRAD's per-iteration statistic; A27)
__host__ __device__ inline float srad_q0sqr(double s, double ss, int64_t n) {
  const double mean = s / (double)n;
  const double var = ss / (double)n - mean * mean;
  return (float)(var / (mean * mean));
}

// ---- SRAD kernel 2: (c, I) -> I' (Rodinia v3.1 srad; A18) --------
template <class AccC, class AccI>
__device__ __forceinline__ acc_value_t<AccI> op_srad2(const AccC& C, const AccI& I, const float* prm) {
  using V = acc_value_t<AccI>;
  const V Ic = I.template at<0, 0, 0>();
  const V dN = vsub(I.template at<0, -1, 0>(), Ic);
  const V dS = vsub(I.template at<0, 1, 0>(), Ic);
  const V dW = vsub(I.template at<0, 0, -1>(), Ic);
  const V dE = vsub(I.template at<0, 0, 1>(), Ic);
  const V cC = C.template at<0, 0, 0>();
  const V cS = C.template at<0, 1, 0>();
  const V cE = C.template at<0, 0, 1>();
  V D = vmul(cC, dN);
  D = vfma(cS, dS, D);
  D = vfma(cC, dW, D);
  D = vfma(cE, dE, D);
  return vfma(vbc<V>(__fmul_rn(0.25f, prm[0])), D, Ic);
}

// ---- Hotspot2D (Rodinia v3.1 hotspot; A26) -----------------------
// T' = T + sdc * (P + (S + N - 2T)*Ry_1 + (E + W - 2T)*Rx_1 + (amb - T)*Rz_1)
template <class AccT, class AccP>
__device__ __forceinline__ float op_hotspot2d(const AccT& T, const AccP& P, const float* prm) {
  const float sdc = prm[0], rx1 = prm[1], ry1 = prm[2], rz1 = prm[3], amb = prm[4];
  const float Tc = T.template at<0, 0, 0>();
  const float a = __fmaf_rn(-2.0f, Tc, __fadd_rn(T.template at<0, 1, 0>(), T.template at<0, -1, 0>()));
  const float b = __fmaf_rn(-2.0f, Tc, __fadd_rn(T.template at<0, 0, 1>(), T.template at<0, 0, -1>()));
  float acc = P.template at<0, 0, 0>();
  acc = __fmaf_rn(a, ry1, acc);
  acc = __fmaf_rn(b, rx1, acc);
  acc = __fmaf_rn(__fsub_rn(amb, Tc), rz1, acc);
  return __fmaf_rn(sdc, acc, Tc);
}

// ---- Gradient (Rawat et al. [36] 2D gradient; A25) ---------------
// out = I + 1/sqrt(eps + (I-N)^2 + (I-S)^2 + (I-W)^2 + (I-E)^2)
template <class Acc>
__device__ __forceinline__ float op_gradient(const Acc& I, const float* prm) {
  const float eps = prm[0];
  const float Ic = I.template at<0, 0, 0>();
  const float d1 = __fsub_rn(Ic, I.template at<0, -1, 0>());
  const float d2 = __fsub_rn(Ic, I.template at<0, 1, 0>());
  const float d3 = __fsub_rn(Ic, I.template at<0, 0, -1>());
  const float d4 = __fsub_rn(Ic, I.template at<0, 0, 1>());
  float s = __fmaf_rn(d1, d1, eps);
  s = __fmaf_rn(d2, d2, s);
  s = __fmaf_rn(d3, d3, s);
  s = __fmaf_rn(d4, d4, s);
  return __fadd_rn(Ic, rsqrt_nr(s));
}

// ---- Acoustic (Listing 3; A19/A20) --------------------
// next = cf(K,l1) * ((2 - l2*K)*u_c + l2*sum_nbr u - cf(K,l2loss)*prev)
// Neighbours are summed in row-major tap order (Listing 3 lines 5-6).
template <int R, class Acc>
__device__ __forceinline__ float acoustic_sum(const Acc& U) {
  float s;
  if constexpr (R == 1) {
    s = U.template at<-1, 0, 0>();
    s = __fadd_rn(s, U.template at<0, -1, 0>());
    s = __fadd_rn(s, U.template at<0, 0, -1>());
    s = __fadd_rn(s, U.template at<0, 0, 1>());
    s = __fadd_rn(s, U.template at<0, 1, 0>());
    s = __fadd_rn(s, U.template at<1, 0, 0>());
  } else {
    s = U.template at<-2, 0, 0>();
    s = __fadd_rn(s, U.template at<-1, 0, 0>());
    s = __fadd_rn(s, U.template at<0, -2, 0>());
    s = __fadd_rn(s, U.template at<0, -1, 0>());
    s = __fadd_rn(s, U.template at<0, 0, -2>());
    s = __fadd_rn(s, U.template at<0, 0, -1>());
    s = __fadd_rn(s, U.template at<0, 0, 1>());
    s = __fadd_rn(s, U.template at<0, 0, 2>());
    s = __fadd_rn(s, U.template at<0, 1, 0>());
    s = __fadd_rn(s, U.template at<0, 2, 0>());
    s = __fadd_rn(s, U.template at<1, 0, 0>());
    s = __fadd_rn(s, U.template at<2, 0, 0>());
  }
  return s;
}

// Number of star neighbours (+-1..+-R per axis) inside the global domain
// (computeNumNeighbors): generated on the fly, 0 bytes.
template <int R, class Int>
__device__ __forceinline__ int acoustic_K(Int gz, Int gy, Int gx, Int nz, Int ny, Int nx) {
  int K = 0;
#pragma unroll
  for (int off = 1; off <= R; ++off) {
    K += (gz - off >= 0) + (gz + off < nz);
    K += (gy - off >= 0) + (gy + off < ny);
    K += (gx - off >= 0) + (gx + off < nx);
  }
  return K;
}

// the point update given the ordered neighbour sum s and the centre uc
template <int R>
__device__ __forceinline__ float acoustic_combine(float s, float uc, float prev, int K, const float* prm) {
  const float l2 = prm[0], loss1 = prm[1], loss2 = prm[2];
  constexpr int kmax = 6 * R;
  const float cf1 = K < kmax ? loss1 : 1.0f;
  const float cf2 = K < kmax ? loss2 : 1.0f;
  float t = __fmul_rn(__fsub_rn(2.0f, __fmul_rn(l2, (float)K)), uc);
  t = __fmaf_rn(l2, s, t);
  t = __fmaf_rn(-cf2, prev, t);
  return __fmul_rn(cf1, t);
}

template <int R, class Acc>
__device__ __forceinline__ float op_acoustic(const Acc& U, float prev, int K, const float* prm) {
  return acoustic_combine<R>(acoustic_sum<R>(U), U.template at<0, 0, 0>(), prev, K, prm);
}

}  // namespace lift

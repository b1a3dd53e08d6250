// kernel_sweep3d.cu — K2: the 3D stencil as a 2.5D sweep along z.
//
// slide_3 over a 3D grid: each CTA owns a 128 x TY tile of the
// (y, x) plane and a chunk of consecutive output planes.  It streams the
// input planes z-R .. z_end+R-1 through a ring of S shared-memory stages: one
// elected producer thread issues one TMA tensor load per plane (a halo'd box
// of (128+8) x (TY+2R) floats: x from x0-4 so the centre columns stay 16-B
// aligned; y from y0-R), completing on the stage's mbarrier; 8 consumer warps
// compute output plane z from stages z-R..z+R as soon as stage z+R lands,
// then release stage z-R.  This is overlapped tiling with the
// overlap size-step = 2R, staged in local (shared) memory, with
// the z-overlap reused through the ring instead of re-read.
//
// Inside a plane, lane l of warp w owns 4 consecutive x outputs of TY/8 rows:
// the in-row neighbourhood comes from the neighbouring lanes' float4 through
// warp shuffles (lanes 0/31 read the halo columns), the y and z neighbours
// are 128-bit shared loads, and the 4 results leave as one st.global.v4.
//
// pad is folded into the loads: the producer remaps the plane
// index (h on z, or "constant plane" without a load); TMA zero-fills the
// (y, x) cells outside the grid, and only edge tiles rewrite those halo cells
// in shared memory with h-remapped values (or pad_value) before use.  The
// neighbourhood function goes through ops.cuh, so every output has the bits
// K0 computes.
#include <cuda.h>
#include <cuda_runtime.h>

#include <mutex>
#include <string>

#include "common.cuh"
#include "launch.hpp"
#include "halo.cuh"
#include "ops.cuh"
#include "tma.cuh"

namespace lift {
namespace {

constexpr int TX = 128;        // outputs per tile row: 32 lanes x float4
constexpr int XH = 4;          // halo columns loaded on each side (>= R, keeps 16-B alignment)
constexpr int BX = TX + 2 * XH;
constexpr int NW = 8;          // consumer warps
constexpr int NCONS = NW * 32;
constexpr unsigned FULL = 0xffffffffu;

enum K2Op { K2_WSTAR = 0, K2_HOTSPOT = 1, K2_ACOUSTIC = 2 };

template <int R, int RPW, int S>
struct Cfg {
  static constexpr int TY = NW * RPW;
  static constexpr int BY = TY + 2 * R;
  static constexpr int TX_BYTES = BX * BY * 4;                         // bytes one TMA box delivers
  static constexpr int STAGE_FLOATS = ((TX_BYTES + 127) / 128) * 128 / 4;
  static constexpr int SMEM = S * STAGE_FLOATS * 4 + 2 * S * 8 + 128;  // + barriers + align slack
};

// Registers holding one output row's neighbourhood for the 4 x-outputs of a lane.
template <int R>
struct Win {
  float x[4 + 2 * R];   // centre row, x offsets -R .. 3+R
  float ym[R][4];       // ym[k-1][i]: y - k
  float yp[R][4];
  float zm[R][4];       // zm[k-1][i]: z - k
  float zp[R][4];
};

template <int R, int I>
struct WinAcc {
  const Win<R>& w;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert((DZ != 0) + (DY != 0) + (DX != 0) <= 1, "star access only");
    if constexpr (DZ < 0) return w.zm[-DZ - 1][I];
    else if constexpr (DZ > 0) return w.zp[DZ - 1][I];
    else if constexpr (DY < 0) return w.ym[-DY - 1][I];
    else if constexpr (DY > 0) return w.yp[DY - 1][I];
    else return w.x[I + R + DX];
  }
};

__device__ __forceinline__ void set4(float (&d)[4], float4 v) {
  d[0] = v.x; d[1] = v.y; d[2] = v.z; d[3] = v.w;
}

template <int OP, int R, int I>
__device__ __forceinline__ float eval(const StencilParams& p, const Win<R>& w, const float (&pw)[4], int64_t gz,
                                      int64_t gy, int64_t gx0) {
  WinAcc<R, I> a{w};
  if constexpr (OP == K2_WSTAR) {
    return op_weighted<R, R, R, true>(a, p.wbox);
  } else if constexpr (OP == K2_HOTSPOT) {
    return op_hotspot3d(a, pw[I], p.prm);
  } else {
    const int K = acoustic_K<R>(gz, gy, gx0 + I, p.gnz, p.n[1], p.n[2]);
    return op_acoustic<R>(a, pw[I], K, p.prm);
  }
}

template <int OP, int R, int RPW, int S>
__global__ void __launch_bounds__(NCONS + 32)
    k2_sweep(const __grid_constant__ StencilParams p, const __grid_constant__ CUtensorMap tmap,
             const float* __restrict__ src, const float* pw_in, float* out, int ntx, int nty, int zc) {
  using C = Cfg<R, RPW, S>;
  constexpr int TY = C::TY;
  extern __shared__ __align__(128) unsigned char smem_raw[];
  float* stages = reinterpret_cast<float*>((reinterpret_cast<uintptr_t>(smem_raw) + 127) & ~uintptr_t(127));
  uint64_t* full = reinterpret_cast<uint64_t*>(stages + S * C::STAGE_FLOATS);
  uint64_t* empty = full + S;

  const int ntile = ntx * nty;
  const int tile = blockIdx.x % ntile;
  const int chunk = blockIdx.x / ntile;
  const int x0 = (tile % ntx) * TX;
  const int y0 = (tile / ntx) * TY;
  const int64_t zs = p.reg0 + (int64_t)chunk * zc;
  const int64_t ze = min(zs + (int64_t)zc, p.reg1);
  if (zs >= ze) return;
  const int nzc = (int)(ze - zs);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

  if (threadIdx.x == 0) {
    for (int s = 0; s < S; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NW);
    }
    fence_mbar_init();
  }
  __syncthreads();

  if (warp == NW) {
    // ---------------- producer: one TMA box per input plane ----------------
    if (lane == 0) {
      prefetch_tmap(&tmap);
      const int nload = nzc + 2 * R;
      for (int i = 0; i < nload; ++i) {
        const int s = i % S, k = i / S;
        if (k > 0) mbar_wait(&empty[s], (k - 1) & 1);
        const int64_t lz = plane_of(p, p.z_off + zs - R + i);
        if (lz >= 0) {
          mbar_arrive_expect_tx(&full[s], C::TX_BYTES);
          tma_load_3d(stages + s * C::STAGE_FLOATS, &tmap, &full[s], x0 - XH, y0 - R, (int)lz);
        } else {
          mbar_arrive(&full[s]);   // constant plane (value pad): nothing to load
        }
      }
    }
    return;
  }

  // ---------------- consumers ----------------
  const int64_t nx = p.n[2], ny = p.n[1];
  const bool edge = (x0 == 0) || (x0 + TX + R > nx) || (y0 < R) || (y0 + TY + R > ny);
  const bool zero_fill_ok = p.pad_value == 0.0f && p.kind[1] == PAD_CONSTANT && p.kind[2] == PAD_CONSTANT;
  const bool need_fix = edge && !zero_fill_ok;
  const int64_t out_plane = p.plane;
  const int xo = x0 + 4 * lane;
  const bool x_ok = xo < nx;

  for (int i = 0; i < 2 * R; ++i) mbar_wait(&full[i % S], (i / S) & 1);

  for (int j = 0; j < nzc; ++j) {
    const int inew = j + 2 * R;
    mbar_wait(&full[inew % S], (inew / S) & 1);
    const int64_t z = zs + j;
    const int64_t gz = p.z_off + z;
    const int sc = (j + R) % S;
    float* cst = stages + sc * C::STAGE_FLOATS;
    if (need_fix) {
      fixup_tile<R, R, XH, BX, C::BY, NCONS>(p, cst, src, plane_of(p, gz), x0, y0, threadIdx.x);
      fence_proxy_async_smem();
      named_bar_sync(1, NCONS);
    }
    // which z-neighbour planes are constant (value pad) planes
    bool zconst_m[R], zconst_p[R];
#pragma unroll
    for (int k = 1; k <= R; ++k) {
      zconst_m[k - 1] = plane_of(p, gz - k) < 0;
      zconst_p[k - 1] = plane_of(p, gz + k) < 0;
    }
#pragma unroll
    for (int jj = 0; jj < RPW; ++jj) {
      const int rr = warp * RPW + jj;           // tile row
      const int64_t gy = y0 + rr;
      const int off = (rr + R) * BX + XH + 4 * lane;
      Win<R> w;
      const float4 c = lds128(cst + off);
      const float4 e = lds128(cst + (rr + R) * BX + (lane == 0 ? 0 : TX + XH));
      float l1 = __shfl_up_sync(FULL, c.w, 1);
      float r1 = __shfl_down_sync(FULL, c.x, 1);
      if (lane == 0) l1 = e.w;
      if (lane == 31) r1 = e.x;
      if constexpr (R == 1) {
        w.x[0] = l1; w.x[1] = c.x; w.x[2] = c.y; w.x[3] = c.z; w.x[4] = c.w; w.x[5] = r1;
      } else {
        float l2 = __shfl_up_sync(FULL, c.z, 1);
        float r2 = __shfl_down_sync(FULL, c.y, 1);
        if (lane == 0) l2 = e.z;
        if (lane == 31) r2 = e.y;
        w.x[0] = l2; w.x[1] = l1; w.x[2] = c.x; w.x[3] = c.y; w.x[4] = c.z; w.x[5] = c.w; w.x[6] = r1; w.x[7] = r2;
      }
#pragma unroll
      for (int k = 1; k <= R; ++k) {
        set4(w.ym[k - 1], lds128(cst + off - k * BX));
        set4(w.yp[k - 1], lds128(cst + off + k * BX));
        const float4 zm = zconst_m[k - 1] ? make_float4(p.pad_value, p.pad_value, p.pad_value, p.pad_value)
                                          : lds128(stages + ((j + R - k) % S) * C::STAGE_FLOATS + off);
        const float4 zp = zconst_p[k - 1] ? make_float4(p.pad_value, p.pad_value, p.pad_value, p.pad_value)
                                          : lds128(stages + ((j + R + k) % S) * C::STAGE_FLOATS + off);
        set4(w.zm[k - 1], zm);
        set4(w.zp[k - 1], zp);
      }
      const bool ok = x_ok && gy < ny;
      const int64_t go = (z + p.ghost) * out_plane + gy * nx + xo;
      float pw[4] = {0.f, 0.f, 0.f, 0.f};
      if constexpr (OP != K2_WSTAR) {
        if (ok) set4(pw, ldg128(pw_in + go));
      }
      float4 res;
      res.x = eval<OP, R, 0>(p, w, pw, gz, gy, xo);
      res.y = eval<OP, R, 1>(p, w, pw, gz, gy, xo);
      res.z = eval<OP, R, 2>(p, w, pw, gz, gy, xo);
      res.w = eval<OP, R, 3>(p, w, pw, gz, gy, xo);
      if (ok) stg128(out + go, res);
    }
    __syncwarp();
    if (lane == 0) mbar_arrive(&empty[j % S]);   // plane z-R is no longer needed
  }
}

// ---------------------------------------------------------------------------
// host side
// ---------------------------------------------------------------------------
bool star_weights(const StencilParams& p, int R) {
  const int S = 2 * R + 1;
  for (int kz = 0; kz < S; ++kz)
    for (int ky = 0; ky < S; ++ky)
      for (int kx = 0; kx < S; ++kx) {
        const int nax = (kz != R) + (ky != R) + (kx != R);
        if (nax > 1 && p.wbox[(kz * S + ky) * S + kx] != 0.0f) return false;
      }
  return true;
}

struct Launcher {
  const void* fn;
  int smem;
  int ty;
  int ctas_per_sm;
};

template <int OP, int R, int RPW, int S>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    using C = Cfg<R, RPW, S>;
    auto fn = k2_sweep<OP, R, RPW, S>;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, C::SMEM);
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, NCONS + 32, C::SMEM) != cudaSuccess) occ = 1;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), C::SMEM, C::TY, occ > 0 ? occ : 1};
  });
  return L;
}

Launcher pick(const StencilParams& p) {
  const int R = p.radius;
  if (p.op == OP_WEIGHTED) return R == 1 ? get_launcher<K2_WSTAR, 1, 2, 5>() : get_launcher<K2_WSTAR, 2, 2, 7>();
  if (p.op == OP_HOTSPOT3D) return get_launcher<K2_HOTSPOT, 1, 2, 5>();
  return R == 1 ? get_launcher<K2_ACOUSTIC, 1, 2, 5>() : get_launcher<K2_ACOUSTIC, 2, 2, 7>();
}

// small cache of encoded tensor maps (pointer + geometry)
struct MapEntry {
  const float* base;
  int64_t nx, ny, nz;
  int by;
  CUtensorMap map;
};

bool get_map(const float* base, int64_t nx, int64_t ny, int64_t nz, int by, CUtensorMap* out, std::string* err) {
  thread_local MapEntry cache[8];
  thread_local int next = 0;
  for (auto& e : cache)
    if (e.base == base && e.nx == nx && e.ny == ny && e.nz == nz && e.by == by) {
      *out = e.map;
      return true;
    }
  MapEntry e{base, nx, ny, nz, by, {}};
  if (!encode_tensor_map_3d(&e.map, base, nx, ny, nz, BX, (uint32_t)by, 1, err)) return false;
  cache[next] = e;
  next = (next + 1) % 8;
  *out = e.map;
  return true;
}

}  // namespace

bool sweep3d_supported(const StencilParams& p) {
  const int R = p.radius;
  if (R != 1 && R != 2) return false;
  for (int d = 0; d < 3; ++d)
    if (p.size[d] != 2 * R + 1 || p.lo[d] != R || p.hi[d] != R || p.step[d] != 1) return false;
  if (p.op == OP_WEIGHTED) {
    if (!star_weights(p, R)) return false;
  } else if (p.op == OP_HOTSPOT3D) {
    if (R != 1) return false;
  } else if (p.op != OP_ACOUSTIC) {
    return false;
  }
  if (p.n[2] % 4 != 0) return false;
  if (p.n[2] >= (1ll << 31) || p.n[1] >= (1ll << 31) || p.n[0] + 2 * p.ghost >= (1ll << 31)) return false;
  return true;
}

cudaError_t launch_sweep3d(const StencilParams& p, const float* in0, const float* in1, float* out,
                           cudaStream_t stream, int num_sms, std::string* err) {
  const int64_t nz_reg = p.reg1 - p.reg0;
  if (nz_reg <= 0) return cudaSuccess;
  const Launcher L = pick(p);
  const int R = p.radius;
  // slid input and point-wise input per op (stencil.h input order)
  const float* slid = (p.op == OP_ACOUSTIC) ? in1 : in0;
  const float* pw = (p.op == OP_ACOUSTIC) ? in0 : (p.op == OP_HOTSPOT3D ? in1 : nullptr);
  CUtensorMap map;
  if (!get_map(slid, p.n[2], p.n[1], p.n[0] + 2 * p.ghost, L.ty + 2 * R, &map, err)) return cudaErrorInvalidValue;
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int nty = (int)((p.n[1] + L.ty - 1) / L.ty);
  const int64_t tiles = (int64_t)ntx * nty;
  const int64_t slots = (int64_t)num_sms * L.ctas_per_sm;
  int64_t nchunk = (4 * slots + tiles - 1) / tiles;
  if (nchunk < 1) nchunk = 1;
  int64_t zc = (nz_reg + nchunk - 1) / nchunk;
  if (zc < 4 && nz_reg >= 4) zc = 4;
  nchunk = (nz_reg + zc - 1) / zc;
  const int64_t grid = tiles * nchunk;
  if (grid > 0x7fffffff) return cudaErrorInvalidConfiguration;
  int ntx_i = ntx, nty_i = nty, zc_i = (int)zc;
  void* args[] = {(void*)&p, (void*)&map, (void*)&slid, (void*)&pw, (void*)&out, &ntx_i, &nty_i, &zc_i};
  return cudaLaunchKernel(L.fn, dim3((unsigned)grid), dim3(NCONS + 32), args, (size_t)L.smem, stream);
}

}  // namespace lift

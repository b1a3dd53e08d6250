// kernel_tile2d.cu — K1: the 2D stencil on TMA-staged halo'd tiles.
//
// map_2(f, slide_2(size, step, pad_2(...))) over a 2D
// grid.  The output is cut into 128 x TY tiles (overlapped tiling, P:693-822:
// each tile's input box carries the 2R-wide overlap).  Persistent CTAs (one
// wave: grid = SMs x resident CTAs) take contiguous runs of tiles in
// row-major tile order, so neighbouring tiles — whose boxes overlap — are in
// flight at the same time and the overlap is served by L2.  Per CTA an
// elected producer thread streams the tiles' boxes ((128+8) x (TY+2RY)
// floats per input grid) through an S-stage shared-memory ring with TMA and
// mbarriers; 8 consumer warps each sweep TY/8 output rows down the box,
// keeping the 2RY+1 rows of x-windows in registers (each box row is read from
// shared memory once per warp) and taking the in-row neighbours from the
// adjacent lanes with warp shuffles; 4 outputs per lane leave as one
// st.global.v4.  Edge tiles rewrite their out-of-grid halo cells (halo.cuh)
// before use.  f goes through ops.cuh (bitwise equal to K0).
#include <cuda.h>
#include <cuda_runtime.h>

#include <mutex>
#include <string>

#include "common.cuh"
#include "halo.cuh"
#include "launch.hpp"
#include "ops.cuh"
#include "tma.cuh"

namespace lift {
namespace {

constexpr int TX = 128;
constexpr int XH = 4;
constexpr int BX = TX + 2 * XH;
constexpr int NW = 8;
constexpr int NCONS = NW * 32;
constexpr unsigned FULL = 0xffffffffu;

enum K1Op { K1_WBOX = 0, K1_SRAD1 = 1, K1_SRAD2 = 2 };

template <int RY, int RPW, int S, int NIN>
struct Cfg {
  static constexpr int TY = NW * RPW;
  static constexpr int BY = TY + 2 * RY;
  static constexpr int BOX_BYTES = BX * BY * 4;
  static constexpr int BOX_FLOATS = ((BOX_BYTES + 127) / 128) * 128 / 4;
  static constexpr int STAGE_FLOATS = NIN * BOX_FLOATS;
  static constexpr int SMEM = S * STAGE_FLOATS * 4 + 2 * S * 8 + 128;
};

// x-window of one box row for the 4 outputs of a lane: offsets -RX .. 3+RX
template <int RX>
__device__ __forceinline__ void load_row(const float* row, int lane, float (&xw)[4 + 2 * RX]) {
  const float4 c = lds128(row + XH + 4 * lane);
  const float4 e = lds128(row + (lane == 0 ? 0 : TX + XH));
  const float cv[4] = {c.x, c.y, c.z, c.w};
  const float ev[4] = {e.x, e.y, e.z, e.w};
#pragma unroll
  for (int k = 1; k <= RX; ++k) {
    float l = __shfl_up_sync(FULL, cv[4 - k], 1);     // x - k from the left lane
    float r = __shfl_down_sync(FULL, cv[k - 1], 1);   // x + 3 + k from the right lane
    if (lane == 0) l = ev[4 - k];
    if (lane == 31) r = ev[k - 1];
    xw[RX - k] = l;
    xw[RX + 3 + k] = r;
  }
#pragma unroll
  for (int i = 0; i < 4; ++i) xw[RX + i] = cv[i];
}

// Accessor over the register ring: rows[(DY + RY) slot][I + RX + DX].
template <int RY, int RX, int I>
struct RingAcc {
  const float (*rows)[4 + 2 * RX];   // rows[0..2RY] ordered y-RY .. y+RY
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert(DZ == 0, "2D");
    return rows[DY + RY][I + RX + DX];
  }
};

template <int OP, int RY, int RX, int I>
__device__ __forceinline__ float eval(const StencilParams& p, const float (*a)[4 + 2 * RX],
                                      const float (*b)[4 + 2 * RX]) {
  if constexpr (OP == K1_WBOX) {
    return op_weighted<0, RY, RX, false>(RingAcc<RY, RX, I>{a}, p.wbox);
  } else if constexpr (OP == K1_SRAD1) {
    return op_srad1(RingAcc<RY, RX, I>{a}, p.prm);
  } else {
    return op_srad2(RingAcc<RY, RX, I>{a}, RingAcc<RY, RX, I>{b}, p.prm);   // (c, I)
  }
}

template <int OP, int RY, int RX, int RPW, int S, int NIN>
__global__ void __launch_bounds__(NCONS + 32)
    k1_tile(const __grid_constant__ StencilParams p, const __grid_constant__ CUtensorMap map0,
            const __grid_constant__ CUtensorMap map1, const float* __restrict__ src0,
            const float* __restrict__ src1, float* __restrict__ out, int ntx, int nty) {
  using C = Cfg<RY, RPW, S, NIN>;
  constexpr int TY = C::TY;
  constexpr int W = 4 + 2 * RX;
  extern __shared__ __align__(128) unsigned char smem_raw[];
  float* stages = reinterpret_cast<float*>((reinterpret_cast<uintptr_t>(smem_raw) + 127) & ~uintptr_t(127));
  uint64_t* full = reinterpret_cast<uint64_t*>(stages + S * C::STAGE_FLOATS);
  uint64_t* empty = full + S;

  const int64_t ntiles = (int64_t)ntx * nty;
  const int64_t t0 = ntiles * blockIdx.x / gridDim.x;
  const int64_t t1 = ntiles * (blockIdx.x + 1) / gridDim.x;
  const int nt = (int)(t1 - t0);
  if (nt <= 0) return;
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
    if (lane == 0) {
      prefetch_tmap(&map0);
      if (NIN > 1) prefetch_tmap(&map1);
      for (int i = 0; i < nt; ++i) {
        const int s = i % S, k = i / S;
        if (k > 0) mbar_wait(&empty[s], (k - 1) & 1);
        const int64_t t = t0 + i;
        const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
        float* st = stages + s * C::STAGE_FLOATS;
        mbar_arrive_expect_tx(&full[s], NIN * C::BOX_BYTES);
        tma_load_3d(st, &map0, &full[s], x0 - XH, y0 - RY, 0);
        if constexpr (NIN > 1) tma_load_3d(st + C::BOX_FLOATS, &map1, &full[s], x0 - XH, y0 - RY, 0);
      }
    }
    return;
  }

  const int64_t nx = p.n[2], ny = p.n[1];
  const bool zero_fill_ok = p.pad_value == 0.0f && p.kind[1] == PAD_CONSTANT && p.kind[2] == PAD_CONSTANT;
  for (int i = 0; i < nt; ++i) {
    const int s = i % S;
    mbar_wait(&full[s], (i / S) & 1);
    const int64_t t = t0 + i;
    const int x0 = (int)(t % ntx) * TX, y0 = (int)(t / ntx) * TY;
    float* st = stages + s * C::STAGE_FLOATS;
    const bool edge = (x0 == 0) || (x0 + TX + RX > nx) || (y0 < RY) || (y0 + TY + RY > ny);
    if (edge && !zero_fill_ok) {
      fixup_tile<RY, RX, XH, BX, C::BY, NCONS>(p, st, src0, 0, x0, y0, threadIdx.x);
      if constexpr (NIN > 1) fixup_tile<RY, RX, XH, BX, C::BY, NCONS>(p, st + C::BOX_FLOATS, src1, 0, x0, y0, threadIdx.x);
      fence_proxy_async_smem();
      named_bar_sync(1, NCONS);
    }
    const int xo = x0 + 4 * lane;
    const bool x_ok = xo < nx;
    const int r0 = warp * RPW;   // first output row of this warp (tile-relative)
    // register ring of 2RY+1 box rows, filled as the warp sweeps down
    float ra[2 * RY + 1][W];
    float rb[(NIN > 1) ? 2 * RY + 1 : 1][W];
#pragma unroll
    for (int k = 0; k < 2 * RY; ++k) {
      load_row<RX>(st + (r0 + k) * BX, lane, ra[k]);
      if constexpr (NIN > 1) load_row<RX>(st + C::BOX_FLOATS + (r0 + k) * BX, lane, rb[k]);
    }
#pragma unroll
    for (int jj = 0; jj < RPW; ++jj) {
      // box row of (output row r0+jj) + RY enters the ring
      load_row<RX>(st + (r0 + jj + 2 * RY) * BX, lane, ra[2 * RY]);
      if constexpr (NIN > 1) load_row<RX>(st + C::BOX_FLOATS + (r0 + jj + 2 * RY) * BX, lane, rb[2 * RY]);
      const int64_t gy = y0 + r0 + jj;
      float4 res;
      res.x = eval<OP, RY, RX, 0>(p, ra, rb);
      res.y = eval<OP, RY, RX, 1>(p, ra, rb);
      res.z = eval<OP, RY, RX, 2>(p, ra, rb);
      res.w = eval<OP, RY, RX, 3>(p, ra, rb);
      if (x_ok && gy < ny) stg128(out + gy * nx + xo, res);
      // rotate
#pragma unroll
      for (int k = 0; k < 2 * RY; ++k) {
#pragma unroll
        for (int q = 0; q < W; ++q) {
          ra[k][q] = ra[k + 1][q];
          if constexpr (NIN > 1) rb[k][q] = rb[k + 1][q];
        }
      }
    }
    __syncwarp();
    if (lane == 0) mbar_arrive(&empty[s]);
  }
}

struct Launcher {
  const void* fn;
  int smem;
  int ty;
  int ry;
  int nin;
  int ctas_per_sm;
};

template <int OP, int RY, int RX, int RPW, int S, int NIN>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    using C = Cfg<RY, RPW, S, NIN>;
    auto fn = k1_tile<OP, RY, RX, RPW, S, NIN>;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, C::SMEM);
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, NCONS + 32, C::SMEM) != cudaSuccess) occ = 1;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), C::SMEM, C::TY, RY, NIN, occ > 0 ? occ : 1};
  });
  return L;
}

bool pick(const StencilParams& p, Launcher* L) {
  const int ry = p.lo[1], rx = p.lo[2];
  if (p.op == OP_WEIGHTED) {
    if (ry == 1 && rx == 1) { *L = get_launcher<K1_WBOX, 1, 1, 4, 3, 1>(); return true; }
    if (ry == 2 && rx == 2) { *L = get_launcher<K1_WBOX, 2, 2, 4, 3, 1>(); return true; }
    if (ry == 1 && rx == 2) { *L = get_launcher<K1_WBOX, 1, 2, 4, 3, 1>(); return true; }
    if (ry == 2 && rx == 1) { *L = get_launcher<K1_WBOX, 2, 1, 4, 3, 1>(); return true; }
    return false;
  }
  if (p.op == OP_SRAD1) { *L = get_launcher<K1_SRAD1, 1, 1, 4, 3, 1>(); return true; }
  if (p.op == OP_SRAD2) { *L = get_launcher<K1_SRAD2, 1, 1, 4, 3, 2>(); return true; }
  return false;
}

struct MapEntry {
  const float* base;
  int64_t nx, ny;
  int by;
  CUtensorMap map;
};

bool get_map(const float* base, int64_t nx, int64_t ny, int by, CUtensorMap* out, std::string* err) {
  thread_local MapEntry cache[8];
  thread_local int next = 0;
  for (auto& e : cache)
    if (e.base == base && e.nx == nx && e.ny == ny && e.by == by) {
      *out = e.map;
      return true;
    }
  MapEntry e{base, nx, ny, by, {}};
  if (!encode_tensor_map_3d(&e.map, base, nx, ny, 1, BX, (uint32_t)by, 1, err)) return false;
  cache[next] = e;
  next = (next + 1) % 8;
  *out = e.map;
  return true;
}

}  // namespace

bool tile2d_supported(const StencilParams& p) {
  // canonical 2D plan: dimension 0 is the dummy (extent 1, size 1, no pad)
  if (p.n[0] != 1 || p.size[0] != 1 || p.lo[0] != 0 || p.hi[0] != 0 || p.slab) return false;
  const int ry = p.lo[1], rx = p.lo[2];
  for (int d = 1; d < 3; ++d)
    if (p.step[d] != 1 || p.hi[d] != p.lo[d] || p.size[d] != 2 * p.lo[d] + 1) return false;
  if (ry < 1 || ry > 2 || rx < 1 || rx > 2) return false;
  if (p.op == OP_SRAD1 || p.op == OP_SRAD2) {
    if (ry != 1 || rx != 1) return false;
  } else if (p.op != OP_WEIGHTED) {
    return false;
  }
  if (p.n[2] % 4 != 0) return false;
  if (p.n[2] >= (1ll << 31) || p.n[1] >= (1ll << 31)) return false;
  return true;
}

cudaError_t launch_tile2d(const StencilParams& p, const float* in0, const float* in1, float* out,
                          cudaStream_t stream, int num_sms, std::string* err) {
  Launcher L;
  if (!pick(p, &L)) {
    *err = "tile2d: no instantiation";
    return cudaErrorNotSupported;
  }
  CUtensorMap m0, m1;
  if (!get_map(in0, p.n[2], p.n[1], L.ty + 2 * L.ry, &m0, err)) return cudaErrorInvalidValue;
  if (L.nin > 1) {
    if (!get_map(in1, p.n[2], p.n[1], L.ty + 2 * L.ry, &m1, err)) return cudaErrorInvalidValue;
  } else {
    m1 = m0;
  }
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int nty = (int)((p.n[1] + L.ty - 1) / L.ty);
  const int64_t ntiles = (int64_t)ntx * nty;
  int64_t grid = (int64_t)num_sms * L.ctas_per_sm;
  if (grid > ntiles) grid = ntiles;
  const float* s1 = L.nin > 1 ? in1 : in0;
  void* args[] = {(void*)&p, (void*)&m0, (void*)&m1, (void*)&in0, (void*)&s1, (void*)&out, (void*)&ntx, (void*)&nty};
  return cudaLaunchKernel(L.fn, dim3((unsigned)grid), dim3(NCONS + 32), args, (size_t)L.smem, stream);
}

}  // namespace lift

// hotspot_tb.cu -- Hotspot with temporal blocking (R19).
//
// One launch advances the grid by S <= 8 steps.  A CTA owns an output tile of
// OH x OW = (48 - 2S) x (128 - 2L) cells (L = S rounded up to a multiple of 4)
// and keeps the extended tile
// (+S cells each side: the dependency cone of S five-point steps) in shared
// memory for all S steps, so T and P leave HBM once per S steps.  The method's
// three steps (Fig. 1b, :258-274) map onto the launch as
//   (Ia) perforation: only kept rows of T and P are requested (16-B cp.async);
//   (Ib) reconstruction: skipped rows are rebuilt in shared memory (the
//        paper's local memory, :383-395) by NN or LI from the kept rows
//        (PAPER.md:526-549), an apron of den-1 rows supplying the sources;
//   kernel execution: S unchanged Rodinia steps (ref [2])
//        ping-pong between two shared-memory buffers.
// Only the first step of a launch reads T from memory, so only it sees
// perforated T (reading R19; oracle `tblock`).  P is static: rebuilt once.
// Image borders clamp at every step (rows: the neighbour index clamps to the
// image's first/last row; columns: ghost columns mirror the border column).
// The update is Rodinia's regrouped as c0 T + cy (T_N + T_S) + cx (T_W + T_E)
// + sdc (P + amb/Rz), with the last term per cell in registers (P is static):
// 3 FFMA + 2 FADD per cell-step.  Cells near the tile edge are computed
// from clamped smem neighbours and are wrong, but they lie outside the S-step
// cone of the OH x OW cells that are stored.
#include <cuda_runtime.h>

#include <cstdint>

#include "hotspot_tb.cuh"
#include "ptx.cuh"

namespace kp {

constexpr int TB_EW = 128, TB_EH = 48, TB_WARPS = 8, TB_RPW = TB_EH / TB_WARPS;  // extended tile; rows per warp
constexpr unsigned TB_FULL = 0xFFFFFFFFu;

__device__ __forceinline__ bool tb_kept(const TBParams& q, int y) {
  if (!q.row_scheme) return true;
  const int t = y % q.den;
  return q.keep_one ? t == 0 : t != q.den - 1;
}

__device__ __forceinline__ float4 ld4(const float* p) { return *reinterpret_cast<const float4*>(p); }
__device__ __forceinline__ void st4(float* p, float4 v) { *reinterpret_cast<float4*>(p) = v; }
__device__ __forceinline__ float el(const float4& v, int k) { return k == 0 ? v.x : k == 1 ? v.y : k == 2 ? v.z : v.w; }
__device__ __forceinline__ void set_el(float4& v, int k, float s) {
  v.x = k == 0 ? s : v.x;
  v.y = k == 1 ? s : v.y;
  v.z = k == 2 ? s : v.z;
  v.w = k == 3 ? s : v.w;
}

// (Ib) rebuild the skipped rows [r0, r1) of T (buffer X) and P (buffer Y) in
// place; lane = one float4.  kmask bit r = smem row r is a kept in-image row,
// so the nearest loaded rows above / below are bit scans (the same sources as
// the mask-phase definition: the nearest kept rows inside the image,
// PAPER.md:539-549).
__device__ __forceinline__ float4 tb_lerp(float4 a, float4 b, float wa) {
  return make_float4(fmaf(a.x - b.x, wa, b.x), fmaf(a.y - b.y, wa, b.y), fmaf(a.z - b.z, wa, b.z),
                     fmaf(a.w - b.w, wa, b.w));
}
__device__ __forceinline__ void tb_rebuild(const TBParams& q, float* X, float* Y, uint64_t kmask, int gy0, int r0,
                                           int r1) {
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  for (int r = r0 + warp; r < r1; r += TB_WARPS) {
    const int gy = gy0 + r;
    if (gy < 0 || gy >= q.Hg || ((kmask >> r) & 1)) continue;
    const uint64_t lo = kmask & ((1ull << r) - 1), hi = kmask >> (r + 1);
    const bool ha = lo != 0, hb = hi != 0;
    const int ra = ha ? 63 - __clzll((long long)lo) : r, rb = hb ? r + __ffsll((long long)hi) : r;
    const int da = r - ra, db = rb - r;
    const int oa = ra * TB_EW + 4 * lane, ob = rb * TB_EW + 4 * lane, o = r * TB_EW + 4 * lane;
    if (q.li && ha && hb) {  // b + (a - b) * db / (da + db): the row kernel's arithmetic
      const float wa = __fdiv_rn((float)db, (float)(da + db));
      st4(X + o, tb_lerp(ld4(X + oa), ld4(X + ob), wa));
      st4(Y + o, tb_lerp(ld4(Y + oa), ld4(Y + ob), wa));
    } else {  // nearest loaded row, ties to the lower row (R6)
      const int os = (!hb || (ha && da <= db)) ? oa : ob;
      st4(X + o, ld4(X + os));
      st4(Y + o, ld4(Y + os));
    }
  }
}

// one step of this warp's rows: T' = c0 T + cy (T_N + T_S) + cx (T_W + T_E) + pc
// (Rodinia regrouped; pc = sdc (P + amb / Rz) per cell).  GHOST: the tile holds
// an image column border (ghost columns mirror it); CLAMPY: one of the rows is
// the image's first / last row (its vertical neighbour clamps to itself).
struct TBStep {
  float c0, cx, cy;
  int rlo, rhi, NR, gl_lane, gr_lane, gr_el, gs_lane, gs_el;
  bool has_l, has_r;
};
template <bool GHOST, bool CLAMPY>
__device__ __forceinline__ void tb_rows(const TBStep& k, const float* src, float* dst, int rbase, int lane,
                                        const float4 (&pc)[TB_RPW]) {
  const f2 c0 = splat2(k.c0), cx = splat2(k.cx), cy = splat2(k.cy);
  float4 tn = ld4(src + max(rbase - 1, 0) * TB_EW + 4 * lane);
  float4 t = ld4(src + rbase * TB_EW + 4 * lane);
#pragma unroll
  for (int j = 0; j < TB_RPW; ++j) {
    const int r = rbase + j;
    float4 ts = ld4(src + min(r + 1, k.NR - 1) * TB_EW + 4 * lane);
    if (CLAMPY) {
      if (r == k.rlo) tn = t;
      if (r == k.rhi) ts = t;
    }
    const float wl = __shfl_up_sync(TB_FULL, t.w, 1);    // lane 0: tile edge (outside the cone)
    const float er = __shfl_down_sync(TB_FULL, t.x, 1);  // lane 31: likewise
    const f2 sy0 = add2(pk2(tn.x, tn.y), pk2(ts.x, ts.y)), sy1 = add2(pk2(tn.z, tn.w), pk2(ts.z, ts.w));
    const f2 sx0 = pk2(wl + t.y, t.x + t.z), sx1 = pk2(t.y + t.w, t.z + er);
    float4 nv;
    up2(fma2(c0, pk2(t.x, t.y), fma2(cy, sy0, fma2(cx, sx0, pk2(pc[j].x, pc[j].y)))), nv.x, nv.y);
    up2(fma2(c0, pk2(t.z, t.w), fma2(cy, sy1, fma2(cx, sx1, pk2(pc[j].z, pc[j].w)))), nv.z, nv.w);
    if (GHOST) {
      const float vl = __shfl_down_sync(TB_FULL, nv.x, 1);
      const float vr = __shfl_sync(TB_FULL, el(nv, k.gs_el), k.gs_lane & 31);
      if (k.has_l && lane == k.gl_lane) nv.w = vl;
      if (k.has_r && lane == k.gr_lane) set_el(nv, k.gr_el, vr);
    }
    st4(dst + r * TB_EW + 4 * lane, nv);
    tn = t;
    t = ts;
  }
}

// CTA = 8 warps; lane l owns extended-tile columns 4l..4l+3 (one float4), warp w
// rows apron + 6w .. +5.  Extended tile = 128 columns x 48 rows: the output
// tile OW x OH = (128 - 2L) x (48 - 2S), L = S rounded up to 4 (16-B alignment).
// Image borders: rows clamp explicitly; columns through ghost columns (global
// -1 and W) that mirror the border column after every step.
__global__ void __launch_bounds__(32 * TB_WARPS, 3) hotspot_tb_kernel(const __grid_constant__ TBParams q) {
  extern __shared__ __align__(16) float sm[];
  const int S = q.steps, L = (S + 3) & ~3;
  const int NR = TB_EH + 2 * q.apron;
  float* A = sm;
  float* B = sm + NR * TB_EW;
  const int tx = blockIdx.x % q.tiles_x, ty = blockIdx.x / q.tiles_x;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int gxb = tx * q.OW - L;                        // global column of smem column 0 (multiple of 4)
  const int gy0 = q.y_begin + ty * q.OH - S - q.apron;  // global row of smem row 0
  const int ya0 = max(0, q.avail0), ya1 = min(q.Hg, q.avail1);

  // kept in-image rows of the tile as a bit mask (NR <= 62): two modulos per lane
  uint64_t kmask;
  {
    const int g0 = gy0 + lane, g1 = gy0 + lane + 32;
    const bool k0 = lane < NR && g0 >= 0 && g0 < q.Hg && tb_kept(q, g0);
    const bool k1 = lane + 32 < NR && g1 >= 0 && g1 < q.Hg && tb_kept(q, g1);
    kmask = (uint64_t)__ballot_sync(TB_FULL, k0) | ((uint64_t)__ballot_sync(TB_FULL, k1) << 32);
  }
  // (Ia) perforated load: kept rows of T -> A and of P -> B, nothing else
  for (int r = warp; r < NR; r += TB_WARPS) {
    const int gy = gy0 + r;
    if (!((kmask >> r) & 1) || gy < ya0 || gy >= ya1) continue;
    const long long roff = (long long)(gy - q.in_row0) * q.W;
    if (q.vec) {  // W % 4 == 0: a 16-B chunk is wholly inside or outside the row
      const int gx = gxb + 4 * lane;
      if (gx >= 0 && gx < q.W) {
        cp_async16(A + r * TB_EW + 4 * lane, q.T + roff + gx);
        cp_async16(B + r * TB_EW + 4 * lane, q.P + roff + gx);
      }
    } else {
#pragma unroll
      for (int k = 0; k < 4; ++k) {
        const int c = lane + 32 * k, gx = gxb + c;
        if (gx >= 0 && gx < q.W) {
          cp_async4(A + r * TB_EW + c, q.T + roff + gx);
          cp_async4(B + r * TB_EW + c, q.P + roff + gx);
        }
      }
    }
  }
  asm volatile("cp.async.wait_all;" ::: "memory");
  __syncthreads();
  if (q.row_scheme) {  // (Ib) reconstruction in shared memory, rows of the extended tile only
    tb_rebuild(q, A, B, kmask, gy0, q.apron, q.apron + TB_EH);
  }
  const int gl = -gxb - 1, gr = q.W - gxb;  // smem columns of the ghost columns (global -1 and W)
  const bool has_l = gl >= 0 && gl < TB_EW, has_r = gr >= 0 && gr < TB_EW;
  __syncthreads();
  if (has_l || has_r) {  // initial ghost columns of T
    for (int r = threadIdx.x; r < NR; r += 32 * TB_WARPS) {
      if (has_l) A[r * TB_EW + gl] = A[r * TB_EW + gl + 1];
      if (has_r) A[r * TB_EW + gr] = A[r * TB_EW + gr - 1];
    }
  }
  // this thread's cells; constant part of the update: sdc * (P + amb / Rz)
  const int rbase = q.apron + warp * TB_RPW;
  const float sdc = q.sdc, pa = q.pamb;
  float4 pc[TB_RPW];
#pragma unroll
  for (int j = 0; j < TB_RPW; ++j) {
    const float4 pv = ld4(B + (rbase + j) * TB_EW + 4 * lane);
    pc[j] = make_float4(fmaf(pv.x, sdc, pa), fmaf(pv.y, sdc, pa), fmaf(pv.z, sdc, pa), fmaf(pv.w, sdc, pa));
  }
  __syncthreads();  // B becomes the ping-pong partner
  TBStep k;
  k.c0 = q.c0;
  k.cx = q.cx;
  k.cy = q.cy;
  k.NR = NR;
  k.rlo = max(0, -gy0);                // smem rows of the image's first / last row
  k.rhi = min(NR - 1, q.Hg - 1 - gy0);
  k.has_l = has_l;
  k.has_r = has_r;
  k.gl_lane = gl >> 2;                 // gl = L - 1 when present: element 3; source: element 0 of the next lane
  k.gr_lane = gr >> 2;
  k.gr_el = gr & 3;
  k.gs_lane = (gr - 1) >> 2;
  k.gs_el = (gr - 1) & 3;
  const bool ghost = has_l || has_r;  // (CTA-uniform)
  const bool clampy = (k.rlo >= rbase && k.rlo < rbase + TB_RPW) || (k.rhi >= rbase && k.rhi < rbase + TB_RPW);
  for (int s = 0; s < S; ++s) {
    const float* src = (s & 1) ? B : A;
    float* dst = (s & 1) ? A : B;
    if (ghost) {
      if (clampy) tb_rows<true, true>(k, src, dst, rbase, lane, pc);
      else tb_rows<true, false>(k, src, dst, rbase, lane, pc);
    } else {
      if (clampy) tb_rows<false, true>(k, src, dst, rbase, lane, pc);
      else tb_rows<false, false>(k, src, dst, rbase, lane, pc);
    }
    __syncthreads();
  }
  // store the OH x OW cells whose S-step cone lies inside the tile
  const float* fin = (S & 1) ? B : A;
  const int gx = gxb + 4 * lane;
  const bool mine = 4 * lane >= L && 4 * lane < L + q.OW;
  for (int e = S + warp; e < S + q.OH; e += TB_WARPS) {
    const int gy = gy0 + q.apron + e;
    if (gy >= q.y_end) break;
    if (!mine) continue;
    const float4 v = ld4(fin + (q.apron + e) * TB_EW + 4 * lane);
    auto put = [&](float* orow) {
      if (q.vec && gx + 3 < q.W) {
        st4(orow + gx, v);
      } else {
#pragma unroll
        for (int k = 0; k < 4; ++k)
          if (gx + k < q.W) orow[gx + k] = el(v, k);
      }
    };
    put(q.out + (long long)(gy - q.out_row0) * q.W);
    // banded: boundary rows also go straight into the neighbours' buffers (NEXT-4)
    if (q.pu && gy < q.y_begin + q.halo_rows) put(q.pu + (long long)(gy - q.pu_row0) * q.W);
    if (q.pd && gy >= q.y_end - q.halo_rows) put(q.pd + (long long)(gy - q.pd_row0) * q.W);
  }
}

// S steps on output rows [y_begin, y_end); returns the launch error
cudaError_t launch_hotspot_tb(TBParams q, cudaStream_t s) {
  constexpr int kMaxDev = 64;  // per device: a process may drive several devices
  static bool attr[kMaxDev] = {};
  int dev = 0;
  cudaGetDevice(&dev);
  if (dev < 0 || dev >= kMaxDev) dev = 0;
  if (!attr[dev]) {
    cudaError_t e = cudaFuncSetAttribute(hotspot_tb_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 227 * 1024);
    if (e != cudaSuccess) return e;
    attr[dev] = true;
  }
  const int L = (q.steps + 3) & ~3;
  q.OW = TB_EW - 2 * L;
  q.OH = TB_EH - 2 * q.steps;
  q.pitch = TB_EW;
  q.tiles_x = (q.W + q.OW - 1) / q.OW;
  const int tiles_y = (q.y_end - q.y_begin + q.OH - 1) / q.OH;
  const size_t smem = (size_t)2 * (TB_EH + 2 * q.apron) * TB_EW * sizeof(float);
  hotspot_tb_kernel<<<q.tiles_x * tiles_y, 32 * TB_WARPS, smem, s>>>(q);
  return cudaGetLastError();
}

}  // namespace kp

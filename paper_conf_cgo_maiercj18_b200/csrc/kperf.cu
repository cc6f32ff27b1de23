// kperf.cu -- the C ABI (include/kperf.h): plan validation, launch geometry,
// Hotspot time loop (single device, banded with NCCL halo exchange, or banded
// on one device for testing), error metric, host-buffer entry point.
#include <cudaTypedefs.h>  // PFN_cuTensorMapEncodeTiled
#include <cuda_runtime.h>
#include <nccl.h>

#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <string>
#include <vector>

#include "../../include/kperf.h"
#include "hotspot_tb.cuh"
#include "p2p.cuh"
#include "kernel.cuh"

namespace kp {
cudaError_t launch_error(int is_u8, const void* exact, const void* approx, long long n, int metric, double* scratch,
                         cudaStream_t s);
size_t error_scratch_doubles();
}  // namespace kp

using kp::KParams;

static thread_local std::string g_err;

static perf_status fail(perf_status st, const std::string& msg) {
  g_err = msg;
  return st;
}
static perf_status cuda_fail(cudaError_t e, const char* where) {
  return fail(PERF_ERR_CUDA, std::string(where) + ": " + cudaGetErrorString(e));
}
#define CK(call)                                        \
  do {                                                  \
    cudaError_t e_ = (call);                            \
    if (e_ != cudaSuccess) return cuda_fail(e_, #call); \
  } while (0)

struct Band {  // banded Hotspot state
  int hb = 0;                 // halo rows each side
  float* buf[2] = {nullptr, nullptr};
  float* pbuf = nullptr;      // power with halo
  unsigned* flags = nullptr;  // NEXT-4 epoch flags: [0] written by the upper band, [1] by the lower band
  void* base = nullptr;       // one allocation: buf0 | buf1 | pbuf | flags (one CUDA IPC handle)
  size_t rows = 0;            // allocated rows (h + 2 hb)
  // NEXT-4 peer links (perf_p2p_attach or bands_local with P2P)
  bool p2p = false;
  float* peer_buf[2][2] = {{nullptr, nullptr}, {nullptr, nullptr}};  // [0 upper / 1 lower band][parity]
  float* peer_pbuf[2] = {nullptr, nullptr};
  unsigned* peer_flag[2] = {nullptr, nullptr};  // my slot in the upper band (its flags[1]) / lower (its flags[0])
  int peer_row0[2] = {0, 0};                    // global row of the neighbours' buffer row 0
  void* peer_ipc[2] = {nullptr, nullptr};       // IPC mappings to close
  unsigned epoch = 0;
};

// byte layout of a band allocation of `rows` x W floats per array
struct BandLayout {
  size_t arr, total;
};
static BandLayout band_layout(size_t rows, size_t W) {
  const size_t arr = (rows * W * sizeof(float) + 255) & ~(size_t)255;
  return {arr, 3 * arr + 256};
}

#ifndef KPERF_CHK_COMPACT
#define KPERF_CHK_COMPACT 1  // compact keep-one checkerboard ring slots (engine.cuh chk_compact)
#endif
static int nin_of(int app) { return app == PERF_APP_HOTSPOT ? 2 : 1; }
#ifndef KPERF_RUNS
#define KPERF_RUNS 0  // auto loader picks TMA bulk runs for column / checker cells (measured 2.5x slower than
                      // 16-B cp.async: one bulk copy per 128-384-B run makes the TMA unit the bound)
#endif
constexpr int kHostChunks = 16;  // perf_run_host: row chunks per call (copy/compute overlap)

struct perf_plan_s {
  int app, W, H, radius, scheme, recon;
  perf_rate rate;
  long long batch = 1, iters = 1, granule_bytes = 128, global_h = -1, band_y0 = 0, tile_w = kp::kNCW, tile_h = 0,
            metric = 0, loader = 0, ring = 0, tile1_w = 16, tile1_h = 16, producer = 0, tblock = 1, p2p = 0,
            overlap = 1, graph = 1, exchange = 1, fold = 1, host_skip = 1;
  unsigned long long gen = 0;  // bumped by every perf_plan_set (graph keys)
  double* d_err = nullptr;
  float* d_tmp = nullptr;
  size_t tmp_elems = 0;
  void* d_stage_in = nullptr;
  void* d_stage_out = nullptr;
  size_t stage_bytes = 0;
  // perf_run_host pipeline: copy-in / copy-out streams and per-chunk events
  cudaStream_t s_in = nullptr, s_out = nullptr;
  cudaEvent_t ev_start = nullptr, ev_done = nullptr;
  cudaEvent_t ev_in[kHostChunks] = {}, ev_c[kHostChunks] = {};
  // ... captured once per (host_in, host_out, staging) into a CUDA graph, so a
  // call is one graph launch instead of ~7 API calls per chunk
  cudaStream_t s_cap = nullptr;
  cudaGraphExec_t g_exec = nullptr;
  const void* g_in = nullptr;
  void* g_out = nullptr;
  void* g_stage = nullptr;
  Band band;
  // banded Hotspot: exchange stream + fork / join events of the overlapped schedule
  cudaStream_t s_x = nullptr;
  cudaEvent_t ev_b = nullptr, ev_x = nullptr;
  // perf_run_hotspot / bands_local: the ITERS loop captured into a CUDA graph
  cudaGraphExec_t hg_exec = nullptr;
  std::vector<const void*> hg_key;
  ncclComm_t comm = nullptr;
  int rank = 0, nranks = 1;
};

static size_t elem_size(int app) { return app == PERF_APP_MEDIAN ? 1 : 4; }

static int next_pow2(int v) {
  int p = 1;
  while (p < v) p <<= 1;
  return p;
}
static int log2i(int v) {
  int l = 0;
  while ((1 << l) < v) ++l;
  return l;
}

// Rodinia Hotspot coefficients, cell size of the 1024 x 1024 chip (R13)
static void hotspot_coeffs(float& sdc, float& rx1, float& ry1, float& rz1, float& amb) {
  const double t_chip = 0.0005, chip = 0.016, gw = chip / 1024.0, gh = chip / 1024.0;
  const double cap = 0.5 * 1.75e6 * t_chip * gw * gh;
  const double rx = gw / (2.0 * 100.0 * t_chip * gh), ry = gh / (2.0 * 100.0 * t_chip * gw);
  const double rz = t_chip / (100.0 * gh * gw);
  const double max_slope = 3.0e6 / (0.5 * t_chip * 1.75e6);
  const double step = 0.001 / max_slope;
  sdc = (float)(step / cap);
  rx1 = (float)(1.0 / rx);
  ry1 = (float)(1.0 / ry);
  rz1 = (float)(1.0 / rz);
  amb = 80.0f;
}

#ifndef KPERF_GS_NCW3
#define KPERF_GS_NCW3 1  // fused pipeline: 3-warp CTAs on whole 768-column strips (make_params)
#endif
#ifndef KPERF_TMA_PROMO
#define KPERF_TMA_PROMO CU_TENSOR_MAP_L2_PROMOTION_L2_128B  // L2 promotion of the TMA cell tiles
#endif
#ifndef KPERF_TMA
#define KPERF_TMA 1  // auto loader: column / keep-one checkerboard cells by one TMA tensor-tile load per row
#endif

// cuTensorMapEncodeTiled through the runtime's driver entry point (no libcuda link)
static PFN_cuTensorMapEncodeTiled_v12000 tma_encoder() {
  static PFN_cuTensorMapEncodeTiled_v12000 fn = nullptr;
  static bool tried = false;
  if (!tried) {
    tried = true;
    void* f = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &f, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(f);
    else
      cudaGetLastError();
  }
  return fn;
}

// the tensor map of a TMA cell load (KParams::tmap): fp32 rows of W, `rows`
// rows (every frame's rows, pitch W), groups of den cells of G columns
static bool encode_tma(KParams& k, const void* in, int W, long long rows) {
  PFN_cuTensorMapEncodeTiled_v12000 enc = tma_encoder();
  if (!enc) return false;
  const cuuint64_t G = (cuuint64_t)k.G, den = (cuuint64_t)k.den, ng = (cuuint64_t)W / (G * den);
  CUresult r;
  if (k.tma_mode == kp::TMA_COL) {
    const cuuint64_t dims[3] = {(cuuint64_t)k.tma_L, ng, (cuuint64_t)rows};
    const cuuint64_t strides[2] = {G * den * 4, (cuuint64_t)W * 4};
    const cuuint32_t box[3] = {(cuuint32_t)k.tma_L, (cuuint32_t)k.tma_ng, 1};
    const cuuint32_t es[3] = {1, 1, 1};
    r = enc(&k.tmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, const_cast<void*>(in), dims, strides, box, es,
            CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, KPERF_TMA_PROMO,
            CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  } else {  // {G, cell, row}, traversal stride den along the cells: every den-th cell from the start cell
    const cuuint64_t dims[3] = {G, ng * den, (cuuint64_t)rows};
    const cuuint64_t strides[2] = {G * 4, (cuuint64_t)W * 4};
    const cuuint32_t box[3] = {(cuuint32_t)G, (cuuint32_t)(k.tma_ng * k.den), 1};
    const cuuint32_t es[3] = {1, (cuuint32_t)k.den, 1};
    r = enc(&k.tmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, const_cast<void*>(in), dims, strides, box, es,
            CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, KPERF_TMA_PROMO,
            CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  }
  return r == CUDA_SUCCESS;
}

// Launch geometry for rows [y_begin, y_end) of `frames` frames (input frame
// pitch: in_frame_rows rows of W, default H).
static perf_status make_params(const perf_plan_s* P, const void* in, const void* in2, void* out, int frames,
                               int in_row0, int avail0, int avail1, int out_row0, int y_begin, int y_end,
                               KParams& k, unsigned& grid, size_t& smem, int in_frame_rows = -1) {
  const int es = (int)elem_size(P->app);
  const int CV = 16 / es;  // elements per 16-B chunk (load / store / alignment unit)
  // elements per consumer lane per row (must match App::V in apps.cuh)
  const int V = P->app == PERF_APP_MEDIAN ? 16 : 8;
  // consumer warps per CTA: 2 for narrow fp32 Gaussian / Sobel images (kernel.cuh)
  const bool narrow = (P->app == PERF_APP_GAUSSIAN || P->app == PERF_APP_SOBEL) && P->W <= 2 * 32 * V;
  // the fused pipeline on whole 768- but not 1024-column strips (C5's 3840): 3 (kernel.cuh)
  const bool gs3 = KPERF_GS_NCW3 && P->app == PERF_APP_GAUSS_SOBEL && P->W % (3 * 32 * V) == 0 && P->W % (4 * 32 * V) != 0;
  const int NCW = narrow ? 2 : (gs3 ? 3 : kp::kNCW);
  const int TW = NCW * 32 * V;
  const int Hg = P->global_h > 0 ? (int)P->global_h : P->H;
  int scheme = P->scheme;
  if (P->rate.num == 0 && scheme != PERF_SCHEME_STENCIL1) scheme = PERF_SCHEME_NONE;
  const bool s1 = scheme == PERF_SCHEME_STENCIL1;
  std::memset(&k, 0, sizeof k);
  k.in = in;
  k.in2 = in2;
  k.out = out;
  k.in_fstride = (long long)P->W * (in_frame_rows > 0 ? in_frame_rows : P->H);
  k.out_fstride = (long long)P->W * P->H;
  k.W = P->W;
  k.ncw = NCW;
  k.Hg = Hg;
  k.in_row0 = in_row0;
  k.avail0 = avail0;
  k.avail1 = avail1;
  k.out_row0 = out_row0;
  k.y_begin = y_begin;
  k.y_end = y_end;
  k.num = (scheme == PERF_SCHEME_NONE || s1) ? 0 : P->rate.num;
  k.den = (scheme == PERF_SCHEME_NONE || s1) ? 1 : P->rate.den;
  k.tile1_w = (int)P->tile1_w;
  k.tile1_h = (int)P->tile1_h;
  k.keep_one = (k.num == k.den - 1) ? 1 : 0;
  const int G = (int)(P->granule_bytes / es);
  k.G = G < 1 ? 1 : G;
  const bool rowwise = scheme == PERF_SCHEME_NONE || scheme == PERF_SCHEME_ROW || s1;  // whole rows kept
  k.fast_ok = (rowwise || (k.G % V) == 0) ? 1 : 0;
  k.fold = (int)P->fold;
  // median, column NN: cells of >= 2 lanes that tile the strip and a warp (kernel.cuh MEDC)
  k.cellmap = (P->app == PERF_APP_MEDIAN && scheme == PERF_SCHEME_COL && P->recon == PERF_RECON_NN && k.den > 1 &&
               k.G % (2 * V) == 0 && k.G <= 32 * V && TW % k.G == 0) ? 1 : 0;
  const bool chunk_uniform = rowwise || (k.G % CV) == 0;
  const bool aligned = ((reinterpret_cast<uintptr_t>(in) | reinterpret_cast<uintptr_t>(out) |
                         reinterpret_cast<uintptr_t>(in2)) & 15) == 0;
  k.vec_io = (P->W % CV == 0) && aligned ? 1 : 0;
  // 256-bit output stores: every lane chunk (V elements, 32 B for fp32) 32-B aligned
  k.vec32 = k.vec_io && es == 4 && (P->W % 8 == 0) && ((reinterpret_cast<uintptr_t>(out) & 31) == 0) &&
            (((size_t)P->W * P->H * es) % 32 == 0) ? 1 : 0;
  // TMA bulk runs of kept cells: cells of whole 16-B chunks, <= 64 cells per tile row (2 run slots per lane)
  const bool runs_ok = k.vec_io && chunk_uniform && (scheme == PERF_SCHEME_COL || scheme == PERF_SCHEME_CHECKER) &&
                       (TW + 2 * ((CV + k.den * k.G + CV - 1) / CV) * CV) / k.G + 2 <= 64;
  // (an explicit TMA request starts as the cp.async cell loader: the slot layout
  // below is chosen for it, then the TMA block switches the loader or refuses)
  int loader = P->loader == kp::L_TMA ? (int)kp::L_ASYNC16 : (int)P->loader;
  if (loader == kp::L_AUTO) {
    if (!k.vec_io) loader = kp::L_SCALAR;
    else if (rowwise) loader = kp::L_BULK;
    else loader = chunk_uniform ? kp::L_ASYNC16 : kp::L_SCALAR;
    // column / checker cells of >= 16 B: TMA bulk copies of kept cell runs, when
    // a row's runs fit the producer's 64 run slots (2 per lane)
    if (loader == kp::L_ASYNC16 && KPERF_RUNS && runs_ok) loader = kp::L_RUNS;
  }
  if (loader == kp::L_RUNS && !runs_ok)
    return fail(PERF_ERR_UNSUPPORTED, "loader RUNS needs the column / checker scheme, aligned 16-B cells, <= 64 cells per tile row");
  if (loader == kp::L_BULK && !(k.vec_io && rowwise))
    return fail(PERF_ERR_UNSUPPORTED, "loader BULK needs the row/none scheme, W % V == 0 and 16-B aligned buffers");
  if (loader == kp::L_ASYNC16 && !(k.vec_io && chunk_uniform))
    return fail(PERF_ERR_UNSUPPORTED, "loader ASYNC16 needs W*sizeof(T) % 16 == 0, aligned buffers, G*sizeof(T) % 16 == 0");
  k.loader = loader;
  // PERF_KEY_PRODUCER 2: bulk rows issued by consumer warp 0 instead of a dedicated
  // producer warp (frees registers for a 5th CTA/SM but refills the ring only once
  // per warp-0 row: measured 5% slower on C2, so the dedicated warp is the default)
  k.inline_prod = (loader == kp::L_BULK && P->producer == 2) ? 1 : 0;
  // halo / apron columns: the lane edge chunk (V) plus, for the column scheme,
  // the distance to the nearest loaded granule on either side (<= den * G)
  int hx = CV;
  if (scheme == PERF_SCHEME_COL) hx = ((CV + k.den * k.G + CV - 1) / CV) * CV;
  k.hx = hx;
  k.row_elems = TW + 2 * hx;
  // keep-one checkerboard (fp32, 16-B cp.async cells, every warp on the fast
  // path): a row keeps 1 cell in den, so its slot holds only those cells,
  // packed -- den x smaller slots, the same ring depth
  // (the consumer reads compact columns only through the phase table, KPERF_CHKTAB;
  // large cells can make the packed slot wider than the full-width one: keep that)
  k.chk_compact = 0;
  const int compact_elems = ((TW / k.G + k.den + 1) / k.den + 1) * k.G;
  if (KPERF_CHK_COMPACT && KPERF_CHKTAB && scheme == PERF_SCHEME_CHECKER && k.keep_one && k.den > 1 && es == 4 &&
      nin_of(P->app) == 1 && loader == kp::L_ASYNC16 && k.fast_ok && k.vec_io && P->W % (32 * V) == 0 &&
      TW % k.G == 0 && hx <= k.G && (k.G * es) % 16 == 0 && TW + 2 * hx <= 32 * 12 * CV &&
      compact_elems < TW + 2 * hx) {
    k.chk_compact = 1;
    k.row_elems = compact_elems;
  }
  // TMA cell loads (fp32, one input, every warp on the fast path): the row's kept
  // cells as one tensor-tile load into a packed slot (engine.cuh producer,
  // kernel.cuh ringcol).  Column scheme: every group of den cells keeps a run of
  // L = (den - num) G columns (skip-one: phases 0..den-2, keep-one: phase 0); the
  // slot holds the strip's groups + one group each side.  Keep-one checkerboard:
  // the compact slots above, one cell per group.  Any shape that does not fit
  // keeps the 16-B cp.async loader.
  k.tma_mode = kp::TMA_NONE;
  {
    const bool want = P->loader == kp::L_TMA || (P->loader == kp::L_AUTO && KPERF_TMA && loader == kp::L_ASYNC16);
    const int gw = k.G * k.den;
    const bool common = es == 4 && nin_of(P->app) == 1 && k.fast_ok && k.vec_io && k.vec32 && P->W % (32 * V) == 0 &&
                        k.den > 1 && gw > 0 && TW % gw == 0 && P->W % gw == 0 && (k.G * es) % 16 == 0 && in != nullptr;
    int mode = kp::TMA_NONE, L = 0, ng = 0;
    if (want && common && scheme == PERF_SCHEME_COL) {
      L = (k.den - k.num) * k.G;
      ng = TW / gw + 2;
      if (L <= 256 && ng <= 256) mode = kp::TMA_COL;
    } else if (want && common && scheme == PERF_SCHEME_CHECKER && k.chk_compact && (TW / k.G) % k.den == 0) {
      L = k.G;
      ng = k.row_elems / k.G;
      if (L <= 256 && ng * k.den <= 256) mode = kp::TMA_CHK;
    }
    if (mode != kp::TMA_NONE) {
      k.tma_mode = mode;
      k.tma_L = L;
      k.tma_ng = ng;
      k.tma_rows_per_frame = (int)(k.in_fstride / P->W);
      if (encode_tma(k, in, P->W, (long long)frames * k.tma_rows_per_frame)) {
        k.loader = loader = kp::L_TMA;
        if (mode == kp::TMA_COL) k.row_elems = ng * L;
        k.row_elems = (k.row_elems + 31) / 32 * 32;  // tensor-tile destinations: 128-B aligned slots
      } else {
        k.tma_mode = kp::TMA_NONE;
      }
    }
    if (P->loader == kp::L_TMA && k.loader != kp::L_TMA)
      return fail(PERF_ERR_UNSUPPORTED,
                  "loader TMA needs fp32 column / keep-one checkerboard cells, W a multiple of 256 and of den * G, "
                  "aligned buffers and a driver with cuTensorMapEncodeTiled");
  }
  // ring: rows a consumer holds for reconstruction + prefetch depth
  int hold = 1;
  if (scheme == PERF_SCHEME_ROW) hold = 2;
  if (scheme == PERF_SCHEME_CHECKER) hold = 2 * (k.keep_one ? k.den - 1 : 1) + 1;  // rows a cell's rebuild spans
  int nr = P->ring > 0 ? next_pow2((int)P->ring) : next_pow2(hold + (hold > 2 ? 4 : 6));
  // fp32 column scheme, skip-one 1/4 and NN 1/2: a 4-row ring (the producer at
  // most 4 rows ahead) measured faster than 8 (C2: Gaussian5 col 1/4 NN 175 ->
  // 162 us, LI 171 -> 164, Sobel3 col 1/4 NN 175 -> 160, col 1/2 NN 153 ->
  // 147 us; LI 1/2 and 3/4 are faster with 8: tools/sweep_ring.py,
  // profiles/r02/sweep_ring_col.txt)
  if (P->ring == 0 && scheme == PERF_SCHEME_COL && es == 4 && k.den > 1 &&
      ((k.den == 4 && P->rate.num == 1) || (k.den == 2 && P->recon == PERF_RECON_NN)))
    nr = 4;
  if (nr < hold + 1) nr = next_pow2(hold + 1);
  const int nin = P->app == PERF_APP_HOTSPOT ? 2 : 1;
  const size_t slot_bytes = (size_t)k.row_elems * nin * es;
  auto bar_bytes = [](int n) { return (size_t)((2 * n * 8 + 127) & ~127); };
  // segment cap (the launcher then picks the wave-filling height below it): Hotspot
  // 64 rows -- its two-input slots + 32-B recipes for 134 rows would leave 2 CTAs/SM
  int seg = (int)(P->tile_h > 0 ? P->tile_h : (nin == 2 ? 64 : 128));
  if (s1) seg = (seg + k.tile1_h - 1) / k.tile1_h * k.tile1_h;  // whole Stencil1 tiles per segment
  // recipes per segment: seg + 2 VR rows, Stencil1: every tile restarts its window
  k.nrec = (s1 ? seg + (seg / k.tile1_h + 1) * 2 * kp::kMaxVR : seg + 2 * kp::kMaxVR) + kp::kRecPad;
  // + the column scheme's per-lane LI weight tables / the checkerboard's phase table
  // (fp32; kernel.cuh ctab: 3 x 32 float4 per consumer warp)
  size_t col_tab = 0;
  if (es == 4 && scheme == PERF_SCHEME_COL) col_tab = (size_t)NCW * 96 * 16;
  if (es == 4 && scheme == PERF_SCHEME_CHECKER) col_tab = (size_t)NCW * 8 * 16;  // den <= 8 int4 phase entries
  const size_t rec_bytes0 = (size_t)NCW * k.nrec * sizeof(kp::Recipe) + col_tab;
  while (nr > next_pow2(hold + 1) && bar_bytes(nr) + nr * slot_bytes + rec_bytes0 > 200 * 1024) nr >>= 1;
  k.nr = nr;
  k.nr_log2 = log2i(nr);
  k.seg_h = seg;
  k.seg_auto = P->tile_h > 0 ? 0 : 1;
  smem = bar_bytes(nr) + (size_t)nr * slot_bytes + rec_bytes0;
  if (smem > 227 * 1024) return fail(PERF_ERR_UNSUPPORTED, "shared-memory ring + recipes exceed 227 KB");
  k.n_strips = (P->W + TW - 1) / TW;
  k.n_segs = (y_end - y_begin + k.seg_h - 1) / k.seg_h;
  k.frames = frames;
  const long long g = (long long)k.n_strips * k.n_segs * frames;
  if (g <= 0 || g > 0x7FFFFFFFLL) return fail(PERF_ERR_INVALID_ARG, "grid size out of range");
  grid = (unsigned)g;
  hotspot_coeffs(k.sdc, k.rx1, k.ry1, k.rz1, k.amb);
  return PERF_OK;
}

static cudaError_t dispatch(const perf_plan_s* P, const KParams& k, unsigned grid, size_t smem, cudaStream_t s) {
  int scheme = (P->rate.num == 0 && P->scheme != PERF_SCHEME_STENCIL1) ? PERF_SCHEME_NONE : P->scheme;
  const int rc = P->recon;
  switch (P->app) {
    case PERF_APP_GAUSSIAN:
      if (k.ncw == 2)
        return P->radius == 1 ? kp::launch_gauss1_n2(scheme, rc, k, grid, smem, s)
                              : kp::launch_gauss2_n2(scheme, rc, k, grid, smem, s);
      return P->radius == 1 ? kp::launch_gauss1(scheme, rc, k, grid, smem, s)
                            : kp::launch_gauss2(scheme, rc, k, grid, smem, s);
    case PERF_APP_SOBEL:
      if (k.ncw == 2)
        return P->radius == 1 ? kp::launch_sobel1_n2(scheme, rc, k, grid, smem, s)
                              : kp::launch_sobel2_n2(scheme, rc, k, grid, smem, s);
      return P->radius == 1 ? kp::launch_sobel1(scheme, rc, k, grid, smem, s)
                            : kp::launch_sobel2(scheme, rc, k, grid, smem, s);
    case PERF_APP_MEDIAN: return kp::launch_median(scheme, rc, k, grid, smem, s);
    case PERF_APP_HOTSPOT: return kp::launch_hotspot(scheme, rc, k, grid, smem, s);
    case PERF_APP_GAUSS_SOBEL:
      return k.ncw == 3 ? kp::launch_gsobel_n3(scheme, rc, k, grid, smem, s) : kp::launch_gsobel(scheme, rc, k, grid, smem, s);
    case PERF_APP_INVERSION: return kp::launch_inversion(scheme, rc, k, grid, smem, s);
  }
  return cudaErrorInvalidValue;
}

static int band_halo(const perf_plan_s* p) {
  // rows an output row at a band edge reads beyond the band: the stencil's
  // vertical radius (Hotspot: radius 1 per step of a launch, TBLOCK steps under
  // temporal blocking; the fused pipeline: 2 + 1) + the distance to the loaded
  // rows a rebuilt row reads (row / checkerboard: < den)
  const bool vertical = p->rate.num > 0 && (p->scheme == PERF_SCHEME_ROW || p->scheme == PERF_SCHEME_CHECKER);
  const int vr = p->app == PERF_APP_HOTSPOT ? (int)p->tblock : (p->app == PERF_APP_GAUSS_SOBEL ? 3 : p->radius);
  return vr + (vertical ? p->rate.den : 0);
}

// temporally blocked Hotspot launch parameters (hotspot_tb.cu) for a plan
static kp::TBParams tb_params(const perf_plan_s* p, const float* T, const float* P, float* out) {
  kp::TBParams q;
  std::memset(&q, 0, sizeof q);
  q.T = T;
  q.P = P;
  q.out = out;
  q.W = p->W;
  q.Hg = p->global_h > 0 ? (int)p->global_h : p->H;
  q.avail1 = q.Hg;
  q.y_end = q.Hg;
  q.row_scheme = (p->rate.num > 0 && p->scheme == PERF_SCHEME_ROW) ? 1 : 0;
  q.den = q.row_scheme ? p->rate.den : 1;
  q.keep_one = q.row_scheme && p->rate.num == p->rate.den - 1;
  q.li = p->recon == PERF_RECON_LINEAR;
  q.apron = q.row_scheme ? q.den - 1 : 0;
  q.vec = (p->W % 4 == 0) && (((reinterpret_cast<uintptr_t>(T) | reinterpret_cast<uintptr_t>(P) |
                                 reinterpret_cast<uintptr_t>(out)) & 15) == 0);
  float sdc, rx1, ry1, rz1, amb;  // regrouped Rodinia coefficients from the same fp32 constants
  hotspot_coeffs(sdc, rx1, ry1, rz1, amb);
  q.sdc = sdc;
  q.cx = (float)((double)sdc * rx1);
  q.cy = (float)((double)sdc * ry1);
  q.c0 = (float)(1.0 - 2.0 * (double)sdc * rx1 - 2.0 * (double)sdc * ry1 - (double)sdc * rz1);
  q.pamb = (float)((double)sdc * amb * rz1);
  return q;
}


extern "C" {

const char* perf_last_error(void) { return g_err.c_str(); }
const char* perf_version(void) { return "kperf 0.1 (sm_100a)"; }

perf_status perf_plan(perf_plan_t* plan, perf_app app, int W, int H, int radius, perf_scheme scheme, perf_rate rate,
                      perf_recon recon) {
  if (!plan) return fail(PERF_ERR_INVALID_ARG, "plan is NULL");
  *plan = nullptr;
  if (app < PERF_APP_GAUSSIAN || app > PERF_APP_INVERSION) return fail(PERF_ERR_INVALID_ARG, "bad app");
  if (scheme < PERF_SCHEME_NONE || scheme > PERF_SCHEME_STENCIL1) return fail(PERF_ERR_INVALID_ARG, "bad scheme");
  if (recon != PERF_RECON_NN && recon != PERF_RECON_LINEAR) return fail(PERF_ERR_INVALID_ARG, "bad recon");
  if (W < 1 || H < 1) return fail(PERF_ERR_INVALID_ARG, "W and H must be >= 1");
  bool r_ok = false;
  switch (app) {
    case PERF_APP_GAUSSIAN:
    case PERF_APP_SOBEL: r_ok = radius == 1 || radius == 2; break;
    case PERF_APP_MEDIAN:
    case PERF_APP_HOTSPOT: r_ok = radius == 1; break;
    case PERF_APP_GAUSS_SOBEL: r_ok = radius == 2; break;
    case PERF_APP_INVERSION: r_ok = radius == 0; break;
  }
  if (!r_ok) return fail(PERF_ERR_INVALID_ARG, "radius not allowed for this app");
  if (rate.den < 1 || rate.den > 8) return fail(PERF_ERR_INVALID_ARG, "rate.den must be in [1, 8]");
  if (!(rate.num == 0 || rate.num == 1 || rate.num == rate.den - 1) || rate.num >= rate.den)
    return fail(PERF_ERR_INVALID_ARG, "rate.num must be 0, 1 or den-1 (and < den)");
  if ((scheme == PERF_SCHEME_NONE || scheme == PERF_SCHEME_STENCIL1) && rate.num != 0)
    return fail(PERF_ERR_INVALID_ARG, "schemes NONE and STENCIL1 need rate.num == 0");
  if (scheme == PERF_SCHEME_STENCIL1 && (app == PERF_APP_HOTSPOT || app == PERF_APP_GAUSS_SOBEL))
    return fail(PERF_ERR_UNSUPPORTED, "STENCIL1 is provided for Gaussian, Sobel, Median and Inversion");
  if (scheme == PERF_SCHEME_CHECKER && rate.num > 0 && H < rate.den)
    return fail(PERF_ERR_INVALID_ARG, "checker scheme needs H >= den");
  perf_plan_s* p = new (std::nothrow) perf_plan_s();
  if (!p) return fail(PERF_ERR_OOM, "host allocation failed");
  p->app = app;
  p->W = W;
  p->H = H;
  p->radius = radius;
  p->scheme = scheme;
  p->recon = recon;
  p->rate = rate;
  p->metric = (app == PERF_APP_SOBEL || app == PERF_APP_GAUSS_SOBEL) ? PERF_METRIC_ME : PERF_METRIC_MRE;
  *plan = p;
  return PERF_OK;
}

static void host_graph_free(perf_plan_s* p);
static void hotspot_graph_free(perf_plan_s* p);

static long long host_h2d_bytes(const perf_plan_s* p);  // (perf_run_host section)

perf_status perf_plan_set(perf_plan_t p, int key, long long v) {
  if (!p) return fail(PERF_ERR_INVALID_ARG, "plan is NULL");
  host_graph_free(p);  // a captured perf_run_host pipeline bakes in the plan's launch parameters
  hotspot_graph_free(p);  // ... and so does a captured Hotspot loop
  ++p->gen;
  switch (key) {
    case PERF_KEY_BATCH:
      if (v < 1) return fail(PERF_ERR_INVALID_ARG, "BATCH must be >= 1");
      p->batch = v;
      return PERF_OK;
    case PERF_KEY_ITERS:
      if (v < 0) return fail(PERF_ERR_INVALID_ARG, "ITERS must be >= 0");
      p->iters = v;
      return PERF_OK;
    case PERF_KEY_GRANULE_BYTES:
      if (v < (long long)elem_size(p->app) || v % (long long)elem_size(p->app) || v > 4096)
        return fail(PERF_ERR_INVALID_ARG, "GRANULE_BYTES must be a positive multiple of sizeof(T), <= 4096");
      p->granule_bytes = v;
      return PERF_OK;
    case PERF_KEY_GLOBAL_H:
      if (v < p->H) return fail(PERF_ERR_INVALID_ARG, "GLOBAL_H must be >= H");
      p->global_h = v;
      return PERF_OK;
    case PERF_KEY_BAND_Y0:
      if (v < 0) return fail(PERF_ERR_INVALID_ARG, "BAND_Y0 must be >= 0");
      p->band_y0 = v;
      return PERF_OK;
    case PERF_KEY_TILE_W:
      if (v != kp::kNCW) return fail(PERF_ERR_UNSUPPORTED, "TILE_W: this build provides 4 consumer warps");
      p->tile_w = v;
      return PERF_OK;
    case PERF_KEY_TILE_H:
      if (v < 1 || v > 4096) return fail(PERF_ERR_INVALID_ARG, "TILE_H must be in [1, 4096]");
      p->tile_h = v;
      return PERF_OK;
    case PERF_KEY_METRIC:
      if (v < 0 || v > 2) return fail(PERF_ERR_INVALID_ARG, "bad METRIC");
      p->metric = v;
      return PERF_OK;
    case PERF_KEY_LOADER:
      if (v < 0 || v > 5) return fail(PERF_ERR_INVALID_ARG, "bad LOADER");
      p->loader = v;
      return PERF_OK;
    case PERF_KEY_RING:
      if (v < 0 || v > 256) return fail(PERF_ERR_INVALID_ARG, "bad RING");
      p->ring = v;
      return PERF_OK;
    case PERF_KEY_HALO_ROWS:
      return fail(PERF_ERR_INVALID_ARG, "HALO_ROWS is read-only");
    case PERF_KEY_CHK_COMPACT:
      return fail(PERF_ERR_INVALID_ARG, "CHK_COMPACT is read-only");
    case PERF_KEY_TILE1_W: {
      const long long vmax = p->app == PERF_APP_MEDIAN ? 512 : 256;
      if (v < 16 || v > vmax || (v & (v - 1)))
        return fail(PERF_ERR_INVALID_ARG, "TILE1_W must be a power of two in [16, 256] (u8: 512)");
      p->tile1_w = v;
      return PERF_OK;
    }
    case PERF_KEY_TILE1_H:
      if (v < 1 || v > 1024) return fail(PERF_ERR_INVALID_ARG, "TILE1_H must be in [1, 1024]");
      p->tile1_h = v;
      return PERF_OK;
    case PERF_KEY_PRODUCER:
      if (v < 0 || v > 2) return fail(PERF_ERR_INVALID_ARG, "PRODUCER must be 0 (auto), 1 (dedicated) or 2 (inline)");
      p->producer = v;
      return PERF_OK;
    case PERF_KEY_TBLOCK:
      if (v < 1 || v > 8) return fail(PERF_ERR_INVALID_ARG, "TBLOCK must be in [1, 8]");
      p->tblock = v;
      return PERF_OK;
    case PERF_KEY_P2P:
      if (v < 0 || v > 1) return fail(PERF_ERR_INVALID_ARG, "P2P must be 0 or 1");
      p->p2p = v;
      return PERF_OK;
    case PERF_KEY_OVERLAP:
      if (v < 0 || v > 1) return fail(PERF_ERR_INVALID_ARG, "OVERLAP must be 0 or 1");
      p->overlap = v;
      return PERF_OK;
    case PERF_KEY_GRAPH:
      if (v < 0 || v > 1) return fail(PERF_ERR_INVALID_ARG, "GRAPH must be 0 or 1");
      p->graph = v;
      return PERF_OK;
    case PERF_KEY_EXCHANGE:
      if (v < 0 || v > 1) return fail(PERF_ERR_INVALID_ARG, "EXCHANGE must be 0 or 1");
      p->exchange = v;
      return PERF_OK;
    case PERF_KEY_FOLD:
      if (v < 0 || v > 1) return fail(PERF_ERR_INVALID_ARG, "FOLD must be 0 or 1");
      p->fold = v;
      return PERF_OK;
    case PERF_KEY_HOST_SKIP:
      if (v < 0 || v > 1) return fail(PERF_ERR_INVALID_ARG, "HOST_SKIP must be 0 or 1");
      p->host_skip = v;
      return PERF_OK;
    case PERF_KEY_H2D_BYTES:
      return fail(PERF_ERR_INVALID_ARG, "H2D_BYTES is read-only");
  }
  return fail(PERF_ERR_INVALID_ARG, "unknown key");
}

perf_status perf_plan_get(perf_plan_t p, int key, long long* v) {
  if (!p || !v) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  switch (key) {
    case PERF_KEY_BATCH: *v = p->batch; return PERF_OK;
    case PERF_KEY_ITERS: *v = p->iters; return PERF_OK;
    case PERF_KEY_GRANULE_BYTES: *v = p->granule_bytes; return PERF_OK;
    case PERF_KEY_GLOBAL_H: *v = p->global_h > 0 ? p->global_h : p->H; return PERF_OK;
    case PERF_KEY_BAND_Y0: *v = p->band_y0; return PERF_OK;
    case PERF_KEY_TILE_W: *v = p->tile_w; return PERF_OK;
    case PERF_KEY_TILE_H: *v = p->tile_h; return PERF_OK;
    case PERF_KEY_METRIC: *v = p->metric; return PERF_OK;
    case PERF_KEY_LOADER: *v = p->loader; return PERF_OK;
    case PERF_KEY_RING: *v = p->ring; return PERF_OK;
    case PERF_KEY_HALO_ROWS: *v = band_halo(p); return PERF_OK;
    case PERF_KEY_TILE1_W: *v = p->tile1_w; return PERF_OK;
    case PERF_KEY_TILE1_H: *v = p->tile1_h; return PERF_OK;
    case PERF_KEY_PRODUCER: *v = p->producer; return PERF_OK;
    case PERF_KEY_TBLOCK: *v = p->tblock; return PERF_OK;
    case PERF_KEY_P2P: *v = p->p2p; return PERF_OK;
    case PERF_KEY_OVERLAP: *v = p->overlap; return PERF_OK;
    case PERF_KEY_GRAPH: *v = p->graph; return PERF_OK;
    case PERF_KEY_EXCHANGE: *v = p->exchange; return PERF_OK;
    case PERF_KEY_FOLD: *v = p->fold; return PERF_OK;
    case PERF_KEY_HOST_SKIP: *v = p->host_skip; return PERF_OK;
    case PERF_KEY_H2D_BYTES: *v = host_h2d_bytes(p); return PERF_OK;
    case PERF_KEY_CHK_COMPACT: {  // the launch geometry perf_run would use on 256-B aligned buffers
      KParams k;
      unsigned grid;
      size_t smem;
      const void* d = reinterpret_cast<const void*>(uintptr_t(1) << 20);
      perf_status st = make_params(p, d, nin_of(p->app) > 1 ? d : nullptr, const_cast<void*>(d), (int)p->batch, 0, 0,
                                   p->H, 0, 0, p->H, k, grid, smem);
      if (st != PERF_OK) return st;
      *v = k.chk_compact;
      return PERF_OK;
    }
  }
  return fail(PERF_ERR_INVALID_ARG, "unknown key");
}

perf_status perf_run(perf_plan_t p, const void* in, void* out, void* stream) {
  if (!p || !in || !out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  if (p->app == PERF_APP_HOTSPOT) return fail(PERF_ERR_INVALID_ARG, "Hotspot runs through perf_run_hotspot");
  if (in == out) return fail(PERF_ERR_INVALID_ARG, "in and out must not alias");
  KParams k;
  unsigned grid;
  size_t smem;
  perf_status st = make_params(p, in, nullptr, out, (int)p->batch, 0, 0, p->H, 0, 0, p->H, k, grid, smem);
  if (st != PERF_OK) return st;
  cudaError_t e = dispatch(p, k, grid, smem, static_cast<cudaStream_t>(stream));
  if (e != cudaSuccess) return cuda_fail(e, "perf_run launch");
  return PERF_OK;
}

static void host_graph_free(perf_plan_s* p) {
  if (p->g_exec) cudaGraphExecDestroy(p->g_exec);
  p->g_exec = nullptr;
  p->g_in = nullptr;
  p->g_out = nullptr;
  p->g_stage = nullptr;
}

static void host_pipe_free(perf_plan_s* p) {
  host_graph_free(p);
  if (p->s_cap) cudaStreamDestroy(p->s_cap);
  p->s_cap = nullptr;
  for (int i = 0; i < kHostChunks; ++i) {
    if (p->ev_in[i]) cudaEventDestroy(p->ev_in[i]);
    if (p->ev_c[i]) cudaEventDestroy(p->ev_c[i]);
    p->ev_in[i] = p->ev_c[i] = nullptr;
  }
  if (p->ev_start) cudaEventDestroy(p->ev_start);
  if (p->ev_done) cudaEventDestroy(p->ev_done);
  if (p->s_in) cudaStreamDestroy(p->s_in);
  if (p->s_out) cudaStreamDestroy(p->s_out);
  p->ev_start = p->ev_done = nullptr;
  p->s_in = p->s_out = nullptr;
}

static cudaError_t host_pipe_init(perf_plan_s* p) {
  if (p->s_in) return cudaSuccess;
  cudaError_t e = cudaStreamCreateWithFlags(&p->s_in, cudaStreamNonBlocking);
  if (e == cudaSuccess && !p->s_cap) e = cudaStreamCreateWithFlags(&p->s_cap, cudaStreamNonBlocking);
  if (e == cudaSuccess) e = cudaStreamCreateWithFlags(&p->s_out, cudaStreamNonBlocking);
  if (e == cudaSuccess) e = cudaEventCreateWithFlags(&p->ev_start, cudaEventDisableTiming);
  if (e == cudaSuccess) e = cudaEventCreateWithFlags(&p->ev_done, cudaEventDisableTiming);
  for (int i = 0; i < kHostChunks && e == cudaSuccess; ++i) {
    e = cudaEventCreateWithFlags(&p->ev_in[i], cudaEventDisableTiming);
    if (e == cudaSuccess) e = cudaEventCreateWithFlags(&p->ev_c[i], cudaEventDisableTiming);
  }
  if (e != cudaSuccess) host_pipe_free(p);
  return e;
}

// perf_run_host, row scheme (HOST_SKIP): which rows cross PCIe
static bool host_row_skip(const perf_plan_s* p) {
  return p->host_skip && p->scheme == PERF_SCHEME_ROW && p->rate.num > 0 && p->rate.den > 1;
}
static bool host_phase_kept(const perf_plan_s* p, int ph) {  // (R2: phase 0 always kept; keep-one keeps phase 0 only)
  return p->rate.num == p->rate.den - 1 ? ph == 0 : ph != p->rate.den - 1;
}
static long long host_h2d_bytes(const perf_plan_s* p) {  // bytes perf_run_host copies in per call
  const long long row = (long long)p->W * (long long)elem_size(p->app);
  long long rows = p->H;
  if (host_row_skip(p)) {
    rows = 0;
    for (int y = 0; y < p->H; ++y) rows += host_phase_kept(p, y % p->rate.den) ? 1 : 0;
  }
  return rows * row * p->batch;
}

// Host-buffer entry: the batch is cut into row chunks (<= kHostChunks); chunk
// i is copied in on s_in and, as soon as it has landed, the kernel computes the
// output rows ending kHostLag rows above its last row (the rows it reads below
// an output row -- stencil radius <= 3 + rebuild apron <= 2 (den - 1) <= 14 --
// are then all in), and those rows are copied out on s_out; PCIe copies in
// both directions overlap each other and the kernels.
static perf_status host_enqueue(perf_plan_s* p, const void* host_in, void* host_out, cudaStream_t s) {
  const size_t es = elem_size(p->app);
  const size_t frame_bytes = (size_t)p->W * p->H * es;
  // chunks: per frame nc row ranges of >= kMinChunkRows rows
  constexpr int kMinChunkRows = 64;  // > kHostLag
  const int B = (int)p->batch, H = p->H;
  // and >= 2 MB per chunk: small frames (C1's 1 MB) are one chunk each
  const size_t row_b = (size_t)p->W * es;
  const int min_rows = std::max(kMinChunkRows, (int)std::min<size_t>((size_t)H, ((size_t)2 << 20) / row_b));
  int nc = std::max(1, std::min(kHostChunks / std::max(B, 1), H / min_rows));
  if (B > kHostChunks) nc = 1;
  const int per = (H + nc - 1) / nc;
  nc = (H + per - 1) / per;
  const size_t row_bytes = (size_t)p->W * es;
  CK(cudaEventRecord(p->ev_start, s));  // order after the caller's earlier work on `stream`
  CK(cudaStreamWaitEvent(p->s_in, p->ev_start, 0));
  CK(cudaStreamWaitEvent(p->s_out, p->ev_start, 0));
  constexpr int kHostLag = 24;  // > radius + rebuild apron of every plan (<= 17)
  // frames beyond kHostChunks chunks reuse events: process in groups
  for (int f0 = 0; f0 < B; f0 += std::max(1, kHostChunks / nc)) {
    const int f1 = std::min(B, f0 + std::max(1, kHostChunks / nc));
    const int n = (f1 - f0) * nc;
    for (int i = 0; i < n; ++i) {  // copy-in
      const int f = f0 + i / nc, c = i % nc, r0 = c * per, r1 = std::min(H, r0 + per);
      if (host_row_skip(p)) {
        // row scheme: only the kept rows cross PCIe -- one strided 2-D copy per
        // kept phase (the kernels never read a skipped row)
        const int den = p->rate.den;
        for (int ph = 0; ph < den; ++ph) {
          if (!host_phase_kept(p, ph)) continue;
          const int y0 = r0 + ((ph - r0) % den + den) % den;
          if (y0 >= r1) continue;
          const int cnt = (r1 - y0 + den - 1) / den;
          const size_t off = (size_t)f * frame_bytes + (size_t)y0 * row_bytes;
          CK(cudaMemcpy2DAsync(static_cast<char*>(p->d_stage_in) + off, den * row_bytes,
                               static_cast<const char*>(host_in) + off, den * row_bytes, row_bytes, cnt,
                               cudaMemcpyHostToDevice, p->s_in));
        }
      } else {
        const size_t off = (size_t)f * frame_bytes + (size_t)r0 * row_bytes;
        CK(cudaMemcpyAsync(static_cast<char*>(p->d_stage_in) + off, static_cast<const char*>(host_in) + off,
                           (size_t)(r1 - r0) * row_bytes, cudaMemcpyHostToDevice, p->s_in));
      }
      CK(cudaEventRecord(p->ev_in[i], p->s_in));
    }
    for (int i = 0; i < n; ++i) {  // compute + copy-out: output rows [r0, r1) lag the input chunk
      const int f = f0 + i / nc, c = i % nc;
      const int r0 = c == 0 ? 0 : c * per - kHostLag, r1 = c == nc - 1 ? H : (c + 1) * per - kHostLag;
      CK(cudaStreamWaitEvent(s, p->ev_in[i], 0));
      KParams k;
      unsigned grid;
      size_t smem;
      const char* fin = static_cast<const char*>(p->d_stage_in) + (size_t)f * frame_bytes;
      char* fout = static_cast<char*>(p->d_stage_out) + (size_t)f * frame_bytes;
      perf_status st = make_params(p, fin, nullptr, fout, 1, 0, 0, H, 0, r0, r1, k, grid, smem);
      if (st != PERF_OK) return st;
      cudaError_t e = dispatch(p, k, grid, smem, s);
      if (e != cudaSuccess) return cuda_fail(e, "perf_run_host launch");
      CK(cudaEventRecord(p->ev_c[i], s));
      CK(cudaStreamWaitEvent(p->s_out, p->ev_c[i], 0));
      const size_t off = (size_t)f * frame_bytes + (size_t)r0 * row_bytes;
      CK(cudaMemcpyAsync(static_cast<char*>(host_out) + off, static_cast<const char*>(p->d_stage_out) + off,
                         (size_t)(r1 - r0) * row_bytes, cudaMemcpyDeviceToHost, p->s_out));
    }
    if (f1 < B) {  // the next group reuses the events: its copies wait for this group's
      CK(cudaEventRecord(p->ev_done, p->s_out));
      CK(cudaStreamWaitEvent(p->s_in, p->ev_done, 0));
      CK(cudaStreamWaitEvent(s, p->ev_done, 0));
    }
  }
  CK(cudaEventRecord(p->ev_done, p->s_out));
  CK(cudaStreamWaitEvent(s, p->ev_done, 0));
  return PERF_OK;
}

static bool is_pinned(const void* ptr) {
  cudaPointerAttributes a;
  if (cudaPointerGetAttributes(&a, ptr) != cudaSuccess) {
    cudaGetLastError();
    return false;
  }
  return a.type == cudaMemoryTypeHost;
}

perf_status perf_run_host(perf_plan_t p, const void* host_in, void* host_out, void* stream) {
  if (!p || !host_in || !host_out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  if (p->app == PERF_APP_HOTSPOT) return fail(PERF_ERR_UNSUPPORTED, "Hotspot has no host-buffer entry point");
  const size_t bytes = (size_t)p->batch * p->W * p->H * elem_size(p->app);
  if (p->stage_bytes < bytes) {
    host_graph_free(p);
    if (p->d_stage_in) cudaFree(p->d_stage_in);
    if (p->d_stage_out) cudaFree(p->d_stage_out);
    p->d_stage_in = p->d_stage_out = nullptr;
    p->stage_bytes = 0;
    if (cudaMalloc(&p->d_stage_in, bytes) != cudaSuccess || cudaMalloc(&p->d_stage_out, bytes) != cudaSuccess)
      return fail(PERF_ERR_OOM, "staging allocation failed");
    p->stage_bytes = bytes;
  }
  CK(host_pipe_init(p));
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  if (!(is_pinned(host_in) && is_pinned(host_out))) {  // pageable: plain enqueue (copies are synchronous anyway)
    perf_status st = host_enqueue(p, host_in, host_out, s);
    if (st != PERF_OK) return st;
    CK(cudaStreamSynchronize(s));
    return PERF_OK;
  }
  if (!(p->g_exec && p->g_in == host_in && p->g_out == host_out && p->g_stage == p->d_stage_in)) {
    host_graph_free(p);
    CK(cudaStreamBeginCapture(p->s_cap, cudaStreamCaptureModeRelaxed));
    perf_status st = host_enqueue(p, host_in, host_out, p->s_cap);
    cudaGraph_t g = nullptr;
    cudaError_t e = cudaStreamEndCapture(p->s_cap, &g);
    if (st != PERF_OK) {
      if (g) cudaGraphDestroy(g);
      return st;
    }
    if (e != cudaSuccess) return cuda_fail(e, "perf_run_host graph capture");
    e = cudaGraphInstantiate(&p->g_exec, g, 0);
    cudaGraphDestroy(g);
    if (e != cudaSuccess) {
      p->g_exec = nullptr;
      return cuda_fail(e, "perf_run_host graph instantiate");
    }
    p->g_in = host_in;
    p->g_out = host_out;
    p->g_stage = p->d_stage_in;
  }
  CK(cudaGraphLaunch(p->g_exec, s));
  CK(cudaStreamSynchronize(s));
  return PERF_OK;
}

// ---------------------------------------------------------------- Hotspot ----
static void band_free(perf_plan_s* p) {
  for (void*& m : p->band.peer_ipc)
    if (m) { cudaIpcCloseMemHandle(m); m = nullptr; }
  if (p->band.base) cudaFree(p->band.base);
  Band fresh;
  p->band = fresh;
}

static perf_status band_alloc(perf_plan_s* p) {
  const int hb = band_halo(p);
  const size_t rows = (size_t)p->H + 2 * hb;
  if (p->band.base && p->band.rows == rows && p->band.hb == hb) return PERF_OK;
  if (p->band.p2p) return fail(PERF_ERR_INVALID_ARG, "band geometry changed after perf_p2p_attach");
  band_free(p);
  const BandLayout L = band_layout(rows, p->W);
  void* base = nullptr;
  if (cudaMalloc(&base, L.total) != cudaSuccess) return fail(PERF_ERR_OOM, "band allocation failed");
  cudaMemset(base, 0, L.total);
  char* b = static_cast<char*>(base);
  p->band.base = base;
  p->band.buf[0] = reinterpret_cast<float*>(b);
  p->band.buf[1] = reinterpret_cast<float*>(b + L.arr);
  p->band.pbuf = reinterpret_cast<float*>(b + 2 * L.arr);
  p->band.flags = reinterpret_cast<unsigned*>(b + 3 * L.arr);
  p->band.rows = rows;
  p->band.hb = hb;
  return PERF_OK;
}

// rows [ya, yb) of one band launch (`steps` Hotspot steps; buffer rows with
// halos) `src` -> `dst`.  pu / pd: NEXT-4 peer stores of the band's first / last
// halo rows (whole-band launches only: the kernels key them off y_begin / y_end)
static perf_status band_launch(perf_plan_s* p, const float* src, float* dst, int steps, int ya, int yb,
                               cudaStream_t s, float* pu = nullptr, float* pd = nullptr) {
  const int Hg = (int)p->global_h, y0 = (int)p->band_y0, h = p->H, hb = p->band.hb;
  if (p->tblock > 1) {  // `steps` steps in one temporally blocked launch
    kp::TBParams q = tb_params(p, src, p->band.pbuf, dst);
    q.pu = pu;
    q.pd = pd;
    q.pu_row0 = p->band.peer_row0[0];
    q.pd_row0 = p->band.peer_row0[1];
    q.halo_rows = hb;
    q.in_row0 = q.out_row0 = y0 - hb;
    q.avail0 = std::max(0, y0 - hb);
    q.avail1 = std::min(Hg, y0 + h + hb);
    q.y_begin = ya;
    q.y_end = yb;
    q.steps = steps;
    cudaError_t e = kp::launch_hotspot_tb(q, s);
    if (e != cudaSuccess) return cuda_fail(e, "hotspot band launch (temporal blocking)");
    return PERF_OK;
  }
  KParams k;
  unsigned grid;
  size_t smem;
  perf_status st = make_params(p, src, p->band.pbuf, dst, 1, y0 - hb, std::max(0, y0 - hb), std::min(Hg, y0 + h + hb),
                               y0 - hb, ya, yb, k, grid, smem);
  if (st != PERF_OK) return st;
  k.in_fstride = k.out_fstride = 0;
  k.pu = pu;
  k.pd = pd;
  k.pu_row0 = p->band.peer_row0[0];
  k.pd_row0 = p->band.peer_row0[1];
  k.halo_rows = hb;
  if (((reinterpret_cast<uintptr_t>(pu) | reinterpret_cast<uintptr_t>(pd)) & 31) != 0) k.vec32 = 0;
  cudaError_t e = dispatch(p, k, grid, smem, s);
  if (e != cudaSuccess) return cuda_fail(e, "hotspot band launch");
  return PERF_OK;
}

// the halo rows of a band (perf_band_halo): the single source of the exchange
// bookkeeping for NCCL, the single-device emulation and the CPU tests
static perf_halo_plan halo_plan(const perf_plan_s* p, int rank) {
  perf_halo_plan h;
  const int hb = band_halo(p), Hg = p->global_h > 0 ? (int)p->global_h : p->H;
  h.halo_rows = hb;
  h.buf_rows = p->H + 2 * hb;
  h.up_rank = p->band_y0 > 0 ? rank - 1 : -1;
  h.down_rank = p->band_y0 + p->H < Hg ? rank + 1 : -1;
  h.send_up_row = hb;         // my first hb rows -> the upper band's bottom halo
  h.recv_up_row = 0;          // its last hb rows -> my top halo
  h.send_down_row = p->H;     // my last hb rows -> the lower band's top halo
  h.recv_down_row = p->H + hb;
  return h;
}

// NCCL halo exchange: `frames` frames of `frame_elems` elements of `es` bytes,
// buffer rows as halo_plan() says; one group (all frames, both neighbours)
static perf_status band_exchange_nccl(perf_plan_s* p, void* buf, size_t es, int frames, size_t frame_elems,
                                      cudaStream_t s) {
  if (!p->exchange || !p->comm) return PERF_OK;
  const perf_halo_plan h = halo_plan(p, p->rank);
  const size_t W = p->W, row_b = W * es, n = (size_t)h.halo_rows * row_b;
  char* b = static_cast<char*>(buf);
  if (ncclGroupStart() != ncclSuccess) return fail(PERF_ERR_NCCL, "ncclGroupStart");
  for (int f = 0; f < frames; ++f) {
    char* fb = b + (size_t)f * frame_elems * es;
    if (h.up_rank >= 0) {
      ncclSend(fb + h.send_up_row * row_b, n, ncclUint8, h.up_rank, p->comm, s);
      ncclRecv(fb + h.recv_up_row * row_b, n, ncclUint8, h.up_rank, p->comm, s);
    }
    if (h.down_rank >= 0) {
      ncclSend(fb + h.send_down_row * row_b, n, ncclUint8, h.down_rank, p->comm, s);
      ncclRecv(fb + h.recv_down_row * row_b, n, ncclUint8, h.down_rank, p->comm, s);
    }
  }
  ncclResult_t r = ncclGroupEnd();
  if (r != ncclSuccess) return fail(PERF_ERR_NCCL, std::string("halo exchange: ") + ncclGetErrorString(r));
  return PERF_OK;
}
static perf_status band_exchange_f32(perf_plan_s* p, float* buf, cudaStream_t s) {
  return band_exchange_nccl(p, buf, sizeof(float), 1, 0, s);
}

// NEXT-4: push my boundary rows of `mine` (buffer rows [hb, 2hb) and [h, h+hb))
// into the neighbours' halos `up`, `dn` (same parity) -- initial T and P only;
// every later halo travels inside the step kernel
static perf_status p2p_push(perf_plan_s* p, const float* mine, float* up, float* dn, cudaStream_t s) {
  const size_t W = p->W, hb = p->band.hb, h = p->H;
  const long long y0 = p->band_y0;
  if (up)
    CK(cudaMemcpyAsync(up + (y0 - p->band.peer_row0[0]) * (long long)W, mine + hb * W, hb * W * sizeof(float),
                       cudaMemcpyDeviceToDevice, s));
  if (dn)
    CK(cudaMemcpyAsync(dn + (y0 + (long long)h - (long long)hb - p->band.peer_row0[1]) * (long long)W, mine + h * W,
                       hb * W * sizeof(float), cudaMemcpyDeviceToDevice, s));
  return PERF_OK;
}
static perf_status p2p_signal(perf_plan_s* p, cudaStream_t s) {
  cudaError_t e = kp::p2p_signal(p->band.peer_flag[0], p->band.peer_flag[1], p->band.epoch + 1, s);
  return e == cudaSuccess ? PERF_OK : cuda_fail(e, "p2p signal");
}
static perf_status p2p_wait(perf_plan_s* p, cudaStream_t s) {
  ++p->band.epoch;
  cudaError_t e = kp::p2p_wait(p->band.flags, p->band.peer_flag[0] != nullptr, p->band.peer_flag[1] != nullptr,
                               p->band.epoch, s);
  return e == cudaSuccess ? PERF_OK : cuda_fail(e, "p2p wait");
}

// exchange stream + fork/join events of the overlapped band schedule
static cudaError_t xstream_init(perf_plan_s* p) {
  if (p->s_x) return cudaSuccess;
  cudaError_t e = cudaStreamCreateWithFlags(&p->s_x, cudaStreamNonBlocking);
  if (e == cudaSuccess) e = cudaEventCreateWithFlags(&p->ev_b, cudaEventDisableTiming);
  if (e == cudaSuccess) e = cudaEventCreateWithFlags(&p->ev_x, cudaEventDisableTiming);
  return e;
}

// The overlapped launch schedule of one band: rows within
// halo_rows of either band edge are computed first; their exchange (`xfer`,
// on the exchange stream) then runs while the interior rows compute; the next
// launch waits for it.  The interior reads only band rows, so it never waits
// for a halo.  `split` false: one whole-band launch, then the exchange.
}  // extern "C" (templates below)

template <class Xfer>
static perf_status band_launch_overlapped(perf_plan_s* p, const float* src, float* dst, int steps, bool split, bool xchg,
                                          cudaStream_t s, Xfer&& xfer) {
  const int y0 = (int)p->band_y0, h = p->H, hb = p->band.hb;
  perf_status st;
  if (!split || !xchg) {
    if ((st = band_launch(p, src, dst, steps, y0, y0 + h, s)) != PERF_OK) return st;
    return xchg ? xfer(s) : PERF_OK;
  }
  if ((st = band_launch(p, src, dst, steps, y0, y0 + hb, s)) != PERF_OK) return st;
  if ((st = band_launch(p, src, dst, steps, y0 + h - hb, y0 + h, s)) != PERF_OK) return st;
  CK(cudaEventRecord(p->ev_b, s));
  CK(cudaStreamWaitEvent(p->s_x, p->ev_b, 0));
  if ((st = xfer(p->s_x)) != PERF_OK) return st;
  CK(cudaEventRecord(p->ev_x, p->s_x));
  if ((st = band_launch(p, src, dst, steps, y0 + hb, y0 + h - hb, s)) != PERF_OK) return st;
  CK(cudaStreamWaitEvent(s, p->ev_x, 0));
  return PERF_OK;
}

extern "C" {

static bool band_splits(const perf_plan_s* p) { return p->overlap && p->H > 2 * band_halo(p); }

// device scratch of perf_run_hotspot (allocated outside any graph capture)
static perf_status hotspot_prepare(perf_plan_s* p, bool banded) {
  const long long n = (long long)p->W * p->H;
  if (!banded && p->iters > 1 && p->tmp_elems < (size_t)n) {
    if (p->d_tmp) cudaFree(p->d_tmp);
    p->d_tmp = nullptr;
    p->tmp_elems = 0;
    if (cudaMalloc(&p->d_tmp, n * sizeof(float)) != cudaSuccess) return fail(PERF_ERR_OOM, "tmp allocation");
    p->tmp_elems = n;
  }
  if (banded) {
    perf_status st = band_alloc(p);
    if (st != PERF_OK) return st;
    if (p->H < p->band.hb) return fail(PERF_ERR_UNSUPPORTED, "band thinner than its halo");
    CK(xstream_init(p));
  }
  return PERF_OK;
}

// the whole ITERS loop of perf_run_hotspot, enqueued on `s` (eager or under capture)
static perf_status hotspot_enqueue(perf_plan_s* p, const float* temp_in, const float* power, float* temp_out,
                                   cudaStream_t s) {
  const long long n = (long long)p->W * p->H;
  const int Hg = p->global_h > 0 ? (int)p->global_h : p->H;
  const bool banded = Hg != p->H || p->band_y0 != 0;
  if (!banded && p->tblock > 1) {  // temporal blocking: one launch per TBLOCK steps
    const long long tb = p->tblock, launches = (p->iters + tb - 1) / tb;
    const float* src = temp_in;
    for (long long l = 0; l < launches; ++l) {
      float* dst = ((launches - 1 - l) % 2 == 0) ? temp_out : p->d_tmp;
      kp::TBParams q = tb_params(p, src, power, dst);
      q.vec = q.vec && ((reinterpret_cast<uintptr_t>(temp_in) | reinterpret_cast<uintptr_t>(temp_out) |
                         reinterpret_cast<uintptr_t>(p->d_tmp)) & 15) == 0;
      q.steps = (int)std::min(tb, p->iters - l * tb);
      cudaError_t e = kp::launch_hotspot_tb(q, s);
      if (e != cudaSuccess) return cuda_fail(e, "hotspot (temporal blocking) launch");
      src = dst;
    }
    return PERF_OK;
  }
  if (!banded) {
    const float* src = temp_in;
    for (long long i = 0; i < p->iters; ++i) {
      float* dst = ((p->iters - 1 - i) % 2 == 0) ? temp_out : p->d_tmp;
      KParams k;
      unsigned grid;
      size_t smem;
      perf_status st = make_params(p, src, power, dst, 1, 0, 0, p->H, 0, 0, p->H, k, grid, smem);
      if (st != PERF_OK) return st;
      cudaError_t e = dispatch(p, k, grid, smem, s);
      if (e != cudaSuccess) return cuda_fail(e, "hotspot launch");
      src = dst;
    }
    return PERF_OK;
  }
  // banded: this rank owns global rows [band_y0, band_y0 + H) of Hg
  const int hb = p->band.hb;
  const size_t W = p->W;
  Band& B = p->band;
  perf_status st;
  CK(cudaMemcpyAsync(B.buf[0] + hb * W, temp_in, n * sizeof(float), cudaMemcpyDeviceToDevice, s));
  CK(cudaMemcpyAsync(B.pbuf + hb * W, power, n * sizeof(float), cudaMemcpyDeviceToDevice, s));
  if (B.p2p) {  // NEXT-4: halos by direct peer stores fused into the step kernels, epoch flags
    if ((st = p2p_push(p, B.buf[0], B.peer_buf[0][0], B.peer_buf[1][0], s)) != PERF_OK) return st;
    if ((st = p2p_push(p, B.pbuf, B.peer_pbuf[0], B.peer_pbuf[1], s)) != PERF_OK) return st;
    if ((st = p2p_signal(p, s)) != PERF_OK || (st = p2p_wait(p, s)) != PERF_OK) return st;
    int cur = 0;
    for (long long i = 0; i < p->iters; i += p->tblock) {
      const int steps = (int)std::min(p->tblock, p->iters - i);
      if ((st = band_launch(p, B.buf[cur], B.buf[cur ^ 1], steps, (int)p->band_y0, (int)p->band_y0 + p->H, s,
                            B.peer_buf[0][cur ^ 1], B.peer_buf[1][cur ^ 1])) != PERF_OK)
        return st;
      if ((st = p2p_signal(p, s)) != PERF_OK || (st = p2p_wait(p, s)) != PERF_OK) return st;
      cur ^= 1;
    }
    CK(cudaMemcpyAsync(temp_out, B.buf[cur] + hb * W, n * sizeof(float), cudaMemcpyDeviceToDevice, s));
    return PERF_OK;
  }
  // NCCL: P once, T before the first launch, then every launch's boundary rows
  // overlapped with its interior (band_launch_overlapped); no exchange after the last
  if ((st = band_exchange_f32(p, B.pbuf, s)) != PERF_OK) return st;
  if ((st = band_exchange_f32(p, B.buf[0], s)) != PERF_OK) return st;
  const bool split = band_splits(p);
  int cur = 0;
  for (long long i = 0; i < p->iters; i += p->tblock) {
    const int steps = (int)std::min(p->tblock, p->iters - i);
    const bool last = i + p->tblock >= p->iters;
    float* dst = B.buf[cur ^ 1];
    if ((st = band_launch_overlapped(p, B.buf[cur], dst, steps, split, !last, s,
                                     [&](cudaStream_t xs) { return band_exchange_f32(p, dst, xs); })) != PERF_OK)
      return st;
    cur ^= 1;
  }
  CK(cudaMemcpyAsync(temp_out, B.buf[cur] + hb * W, n * sizeof(float), cudaMemcpyDeviceToDevice, s));
  return PERF_OK;
}

static void hotspot_graph_free(perf_plan_s* p) {
  if (p->hg_exec) cudaGraphExecDestroy(p->hg_exec);
  p->hg_exec = nullptr;
  p->hg_key.clear();
}

}  // extern "C" (template below)

// capture `enqueue` (which enqueues on the stream it is given) into the plan's
// CUDA graph keyed by `key`, then launch it on `s`; on a capture failure fall
// back to eager launches for this plan (PERF_KEY_GRAPH then reads 2)
template <class Enq>
static perf_status graph_run(perf_plan_s* p, const std::vector<const void*>& key, cudaStream_t s, Enq&& enqueue) {
  if (p->graph != 1) return enqueue(s);
  if (!(p->hg_exec && p->hg_key == key)) {
    hotspot_graph_free(p);
    if (!p->s_cap) CK(cudaStreamCreateWithFlags(&p->s_cap, cudaStreamNonBlocking));
    CK(cudaStreamBeginCapture(p->s_cap, cudaStreamCaptureModeRelaxed));
    perf_status st = enqueue(p->s_cap);
    cudaGraph_t g = nullptr;
    cudaError_t e = cudaStreamEndCapture(p->s_cap, &g);
    if (st != PERF_OK) {
      if (g) cudaGraphDestroy(g);
      return st;
    }
    if (e == cudaSuccess) e = cudaGraphInstantiate(&p->hg_exec, g, 0);
    if (g) cudaGraphDestroy(g);
    if (e != cudaSuccess) {  // e.g. a transport that refuses capture: run eagerly from now on
      cudaGetLastError();
      p->hg_exec = nullptr;
      p->graph = 2;
      return enqueue(s);
    }
    p->hg_key = key;
  }
  CK(cudaGraphLaunch(p->hg_exec, s));
  return PERF_OK;
}

extern "C" {

perf_status perf_run_hotspot(perf_plan_t p, const float* temp_in, const float* power, float* temp_out, void* stream) {
  if (!p || !temp_in || !power || !temp_out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  if (p->app != PERF_APP_HOTSPOT) return fail(PERF_ERR_INVALID_ARG, "plan is not a Hotspot plan");
  if (temp_in == temp_out) return fail(PERF_ERR_INVALID_ARG, "temp_in and temp_out must not alias");
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  const long long n = (long long)p->W * p->H;
  const int Hg = p->global_h > 0 ? (int)p->global_h : p->H;
  const bool banded = Hg != p->H || p->band_y0 != 0;
  if (p->iters == 0) {
    CK(cudaMemcpyAsync(temp_out, temp_in, n * sizeof(float), cudaMemcpyDeviceToDevice, s));
    return PERF_OK;
  }
  if (p->tblock > 1) {
    const bool exact = p->rate.num == 0 || p->scheme == PERF_SCHEME_NONE;
    if (!exact && p->scheme != PERF_SCHEME_ROW) return fail(PERF_ERR_UNSUPPORTED, "TBLOCK > 1 needs the NONE or ROW scheme");
  }
  if (banded && !p->comm && !p->band.p2p && p->nranks == 1 && Hg != p->H)
    return fail(PERF_ERR_INVALID_ARG,
                "banded Hotspot needs perf_comm_init or perf_p2p_attach (or perf_run_hotspot_bands_local)");
  perf_status st = hotspot_prepare(p, banded);
  if (st != PERF_OK) return st;
  auto enq = [&](cudaStream_t cs) { return hotspot_enqueue(p, temp_in, power, temp_out, cs); };
  if (banded && p->band.p2p) return enq(s);  // host-side epoch counters: never replayed from a graph
  return graph_run(p, {temp_in, power, temp_out}, s, enq);
}

/* Single-device emulation of the sharded Hotspot: nb band plans (consecutive
 * bands of one grid) step in lockstep on `stream`, halos copied device to
 * device instead of NCCL (same halo_plan bookkeeping, same overlapped
 * boundary / interior schedule on the exchange stream of plans[0], same graph
 * capture).  temp_in/power/temp_out are whole-grid buffers. */
static perf_status bands_local_enqueue(perf_plan_t* plans, int nb, const float* temp_in, const float* power,
                                       float* temp_out, cudaStream_t s) {
  const size_t W = plans[0]->W;
  const long long iters = plans[0]->iters;
  for (int b = 0; b < nb; ++b) {
    perf_plan_s* p = plans[b];
    const size_t off = (size_t)p->band_y0 * W, n = (size_t)p->H * W, hbw = (size_t)p->band.hb * W;
    CK(cudaMemcpyAsync(p->band.buf[0] + hbw, temp_in + off, n * sizeof(float), cudaMemcpyDeviceToDevice, s));
    CK(cudaMemcpyAsync(p->band.pbuf + hbw, power + off, n * sizeof(float), cudaMemcpyDeviceToDevice, s));
  }
  // band b's halos from its neighbours' boundary rows, rows as halo_plan() says
  auto exchange = [&](int which, bool power_buf, cudaStream_t xs) -> perf_status {
    if (!plans[0]->exchange) return PERF_OK;
    for (int b = 0; b < nb; ++b) {
      perf_plan_s* p = plans[b];
      const perf_halo_plan h = halo_plan(p, b);
      float* mine = power_buf ? p->band.pbuf : p->band.buf[which];
      const size_t rows_b = (size_t)h.halo_rows * W * sizeof(float);
      if (h.up_rank >= 0) {
        perf_plan_s* q = plans[h.up_rank];
        const float* theirs = power_buf ? q->band.pbuf : q->band.buf[which];
        CK(cudaMemcpyAsync(mine + (size_t)h.recv_up_row * W, theirs + (size_t)halo_plan(q, h.up_rank).send_down_row * W,
                           rows_b, cudaMemcpyDeviceToDevice, xs));
      }
      if (h.down_rank >= 0) {
        perf_plan_s* q = plans[h.down_rank];
        const float* theirs = power_buf ? q->band.pbuf : q->band.buf[which];
        CK(cudaMemcpyAsync(mine + (size_t)h.recv_down_row * W, theirs + (size_t)halo_plan(q, h.down_rank).send_up_row * W,
                           rows_b, cudaMemcpyDeviceToDevice, xs));
      }
    }
    return PERF_OK;
  };
  perf_status st;
  const long long tb = plans[0]->tblock;
  if (plans[0]->p2p) {  // NEXT-4 emulated on one device: direct peer stores + epoch flags, no copies
    for (int b = 0; b < nb; ++b) {  // wire neighbours' band buffers as the peers
      Band& B = plans[b]->band;
      if (b > 0) {
        Band& U = plans[b - 1]->band;
        if (U.hb != B.hb) return fail(PERF_ERR_INVALID_ARG, "band plans must share the halo size");
        B.peer_buf[0][0] = U.buf[0];
        B.peer_buf[0][1] = U.buf[1];
        B.peer_pbuf[0] = U.pbuf;
        B.peer_flag[0] = U.flags + 1;
        B.peer_row0[0] = (int)plans[b - 1]->band_y0 - U.hb;
      }
      if (b < nb - 1) {
        Band& D = plans[b + 1]->band;
        B.peer_buf[1][0] = D.buf[0];
        B.peer_buf[1][1] = D.buf[1];
        B.peer_pbuf[1] = D.pbuf;
        B.peer_flag[1] = D.flags;
        B.peer_row0[1] = (int)plans[b + 1]->band_y0 - D.hb;
      }
      B.p2p = true;
    }
    for (int b = 0; b < nb; ++b) {
      Band& B = plans[b]->band;
      if ((st = p2p_push(plans[b], B.buf[0], B.peer_buf[0][0], B.peer_buf[1][0], s)) != PERF_OK) return st;
      if ((st = p2p_push(plans[b], B.pbuf, B.peer_pbuf[0], B.peer_pbuf[1], s)) != PERF_OK) return st;
    }
    // one stream: every band's launch, then every band's signal, then every wait
    auto sync_all = [&]() -> perf_status {
      perf_status r;
      for (int b = 0; b < nb; ++b)
        if ((r = p2p_signal(plans[b], s)) != PERF_OK) return r;
      for (int b = 0; b < nb; ++b)
        if ((r = p2p_wait(plans[b], s)) != PERF_OK) return r;
      return PERF_OK;
    };
    if ((st = sync_all()) != PERF_OK) return st;
    int cur = 0;
    for (long long i = 0; i < iters; i += tb) {
      const int steps = (int)std::min(tb, iters - i);
      for (int b = 0; b < nb; ++b) {
        Band& B = plans[b]->band;
        perf_plan_s* p = plans[b];
        if ((st = band_launch(p, B.buf[cur], B.buf[cur ^ 1], steps, (int)p->band_y0, (int)p->band_y0 + p->H, s,
                              B.peer_buf[0][cur ^ 1], B.peer_buf[1][cur ^ 1])) != PERF_OK)
          return st;
      }
      if ((st = sync_all()) != PERF_OK) return st;
      cur ^= 1;
    }
    for (int b = 0; b < nb; ++b) {
      perf_plan_s* p = plans[b];
      CK(cudaMemcpyAsync(temp_out + (size_t)p->band_y0 * W, p->band.buf[cur] + (size_t)p->band.hb * W,
                         (size_t)p->H * W * sizeof(float), cudaMemcpyDeviceToDevice, s));
      p->band.p2p = false;  // (local wiring is per call)
    }
    return PERF_OK;
  }
  if ((st = exchange(0, true, s)) != PERF_OK) return st;
  if ((st = exchange(0, false, s)) != PERF_OK) return st;
  bool split = true;
  for (int b = 0; b < nb; ++b) split = split && band_splits(plans[b]);
  perf_plan_s* p0 = plans[0];
  int cur = 0;
  for (long long i = 0; i < iters; i += tb) {
    const int steps = (int)std::min(tb, iters - i);
    const bool last = i + tb >= iters;
    if (split && !last) {  // every band's boundary rows, the exchange on p0's stream, every interior
      for (int b = 0; b < nb; ++b) {
        perf_plan_s* p = plans[b];
        const int y0 = (int)p->band_y0, h = p->H, hb = p->band.hb;
        if ((st = band_launch(p, p->band.buf[cur], p->band.buf[cur ^ 1], steps, y0, y0 + hb, s)) != PERF_OK) return st;
        if ((st = band_launch(p, p->band.buf[cur], p->band.buf[cur ^ 1], steps, y0 + h - hb, y0 + h, s)) != PERF_OK)
          return st;
      }
      CK(cudaEventRecord(p0->ev_b, s));
      CK(cudaStreamWaitEvent(p0->s_x, p0->ev_b, 0));
      if ((st = exchange(cur ^ 1, false, p0->s_x)) != PERF_OK) return st;
      CK(cudaEventRecord(p0->ev_x, p0->s_x));
      for (int b = 0; b < nb; ++b) {
        perf_plan_s* p = plans[b];
        const int y0 = (int)p->band_y0, h = p->H, hb = p->band.hb;
        if ((st = band_launch(p, p->band.buf[cur], p->band.buf[cur ^ 1], steps, y0 + hb, y0 + h - hb, s)) != PERF_OK)
          return st;
      }
      CK(cudaStreamWaitEvent(s, p0->ev_x, 0));
    } else {
      for (int b = 0; b < nb; ++b) {
        perf_plan_s* p = plans[b];
        if ((st = band_launch(p, p->band.buf[cur], p->band.buf[cur ^ 1], steps, (int)p->band_y0,
                              (int)p->band_y0 + p->H, s)) != PERF_OK)
          return st;
      }
      if (!last && (st = exchange(cur ^ 1, false, s)) != PERF_OK) return st;
    }
    cur ^= 1;
  }
  for (int b = 0; b < nb; ++b) {
    perf_plan_s* p = plans[b];
    CK(cudaMemcpyAsync(temp_out + (size_t)p->band_y0 * W, p->band.buf[cur] + (size_t)p->band.hb * W,
                       (size_t)p->H * W * sizeof(float), cudaMemcpyDeviceToDevice, s));
  }
  return PERF_OK;
}

perf_status perf_run_hotspot_bands_local(perf_plan_t* plans, int nb, const float* temp_in, const float* power,
                                         float* temp_out, void* stream) {
  if (!plans || nb < 1 || !temp_in || !power || !temp_out) return fail(PERF_ERR_INVALID_ARG, "bad arguments");
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  const size_t W = plans[0]->W;
  const long long iters = plans[0]->iters;
  for (int b = 0; b < nb; ++b) {
    perf_plan_s* p = plans[b];
    if (!p || p->app != PERF_APP_HOTSPOT || (size_t)p->W != W || p->iters != iters || p->tblock != plans[0]->tblock)
      return fail(PERF_ERR_INVALID_ARG, "band plans must be Hotspot plans of one grid (same ITERS, TBLOCK)");
    if (p->tblock > 1 && p->rate.num > 0 && p->scheme != PERF_SCHEME_ROW && p->scheme != PERF_SCHEME_NONE)
      return fail(PERF_ERR_UNSUPPORTED, "TBLOCK > 1 needs the NONE or ROW scheme");
    if (b > 0 && p->band_y0 != plans[b - 1]->band_y0 + plans[b - 1]->H)
      return fail(PERF_ERR_INVALID_ARG, "bands must be consecutive");
    perf_status st = hotspot_prepare(p, true);
    if (st != PERF_OK) return st;
  }
  auto enq = [&](cudaStream_t cs) { return bands_local_enqueue(plans, nb, temp_in, power, temp_out, cs); };
  if (plans[0]->p2p) return enq(s);  // epoch counters live on the host
  std::vector<const void*> key = {temp_in, power, temp_out};
  for (int b = 0; b < nb; ++b) {  // (a perf_plan_set on any band plan changes its gen)
    key.push_back(plans[b]);
    key.push_back(reinterpret_cast<const void*>((uintptr_t)plans[b]->gen));
  }
  return graph_run(plans[0], key, s, enq);
}

static perf_status error_sums(perf_plan_s* p, const void* exact, const void* approx, cudaStream_t s, double h[3]) {
  if (!p->d_err) {
    if (cudaMalloc(&p->d_err, kp::error_scratch_doubles() * sizeof(double)) != cudaSuccess)
      return fail(PERF_ERR_OOM, "error scratch allocation");
  }
  const long long n = (long long)p->batch * p->W * p->H;
  cudaError_t e = kp::launch_error(p->app == PERF_APP_MEDIAN, exact, approx, n, (int)p->metric, p->d_err, s);
  if (e != cudaSuccess) return cuda_fail(e, "perf_error launch");
  CK(cudaMemcpyAsync(h, p->d_err + kp::error_scratch_doubles() - 3, 3 * sizeof(double), cudaMemcpyDeviceToHost, s));
  CK(cudaStreamSynchronize(s));
  return PERF_OK;
}

perf_status perf_error_finish(perf_plan_t p, const double h[3], double* err_out, long long* count_out) {
  if (!p || !h || !err_out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  const long long c = (long long)h[2];
  if (count_out) *count_out = c;
  if (p->metric == PERF_METRIC_ME) *err_out = h[1] > 0 ? h[0] / h[1] : 0.0;
  else *err_out = c > 0 ? h[0] / (double)c : 0.0;
  return PERF_OK;
}

perf_status perf_error_sums(perf_plan_t p, const void* exact, const void* approx, void* stream, double sums[3]) {
  if (!p || !exact || !approx || !sums) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  return error_sums(p, exact, approx, static_cast<cudaStream_t>(stream), sums);
}

perf_status perf_error(perf_plan_t p, const void* exact, const void* approx, void* stream, double* err_out,
                       long long* count_out) {
  if (!p || !exact || !approx || !err_out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  double h[3];
  perf_status st = error_sums(p, exact, approx, static_cast<cudaStream_t>(stream), h);
  if (st != PERF_OK) return st;
  return perf_error_finish(p, h, err_out, count_out);
}

perf_status perf_error_allreduce(perf_plan_t p, const void* exact, const void* approx, void* stream, double* err_out,
                                 long long* count_out) {
  if (!p || !exact || !approx || !err_out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  double h[3];
  perf_status st = error_sums(p, exact, approx, s, h);
  if (st != PERF_OK) return st;
  if (p->comm && p->nranks > 1) {  // (Σ terms, Σ|e|, count) summed over the ranks, in place on the device
    double* d = p->d_err + kp::error_scratch_doubles() - 3;
    ncclResult_t r = ncclAllReduce(d, d, 3, ncclFloat64, ncclSum, p->comm, s);
    if (r != ncclSuccess) return fail(PERF_ERR_NCCL, std::string("error allreduce: ") + ncclGetErrorString(r));
    CK(cudaMemcpyAsync(h, d, sizeof h, cudaMemcpyDeviceToHost, s));
    CK(cudaStreamSynchronize(s));
  }
  return perf_error_finish(p, h, err_out, count_out);
}

perf_status perf_band_halo(perf_plan_t p, int rank, int nranks, perf_halo_plan* out) {
  if (!p || !out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  if (nranks < 1 || rank < 0 || rank >= nranks) return fail(PERF_ERR_INVALID_ARG, "bad rank / nranks");
  *out = halo_plan(p, rank);
  const int Hg = p->global_h > 0 ? (int)p->global_h : p->H;
  if ((p->band_y0 > 0 && rank == 0) || (p->band_y0 + p->H < Hg && rank == nranks - 1) ||
      (p->band_y0 == 0 && rank > 0) || (p->band_y0 + p->H >= Hg && rank < nranks - 1))
    return fail(PERF_ERR_INVALID_ARG, "band geometry (BAND_Y0, H, GLOBAL_H) does not match rank / nranks");
  return PERF_OK;
}

perf_status perf_run_band(perf_plan_t p, void* in_band, void* out, void* stream) {
  if (!p || !in_band || !out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  if (p->app == PERF_APP_HOTSPOT) return fail(PERF_ERR_UNSUPPORTED, "Hotspot bands run through perf_run_hotspot");
  const int Hg = p->global_h > 0 ? (int)p->global_h : p->H, y0 = (int)p->band_y0, h = p->H;
  if (y0 + h > Hg) return fail(PERF_ERR_INVALID_ARG, "band extends below GLOBAL_H");
  if (p->scheme == PERF_SCHEME_STENCIL1 && y0 % (int)p->tile1_h != 0)
    return fail(PERF_ERR_UNSUPPORTED, "STENCIL1 bands must start on a tile row (BAND_Y0 % TILE1_H == 0)");
  cudaStream_t s = static_cast<cudaStream_t>(stream);
  const perf_halo_plan hp = halo_plan(p, p->rank);
  const int hb = hp.halo_rows;
  const size_t es = elem_size(p->app), fin = (size_t)hp.buf_rows * p->W;
  perf_status st = band_exchange_nccl(p, in_band, es, (int)p->batch, fin, s);
  if (st != PERF_OK) return st;
  KParams k;
  unsigned grid;
  size_t smem;
  st = make_params(p, in_band, nullptr, out, (int)p->batch, y0 - hb, std::max(0, y0 - hb), std::min(Hg, y0 + h + hb), y0,
                   y0, y0 + h, k, grid, smem, hp.buf_rows);
  if (st != PERF_OK) return st;
  k.out_fstride = (long long)h * p->W;
  cudaError_t e = dispatch(p, k, grid, smem, s);
  if (e != cudaSuccess) return cuda_fail(e, "perf_run_band launch");
  return PERF_OK;
}

perf_status perf_comm_unique_id(void* out) {
  if (!out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  ncclUniqueId id;
  ncclResult_t r = ncclGetUniqueId(&id);
  if (r != ncclSuccess) return fail(PERF_ERR_NCCL, ncclGetErrorString(r));
  std::memcpy(out, &id, sizeof id);
  return PERF_OK;
}

perf_status perf_comm_init(perf_plan_t p, const void* uid, int rank, int nranks) {
  if (!p || !uid) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  if (nranks < 1 || rank < 0 || rank >= nranks) return fail(PERF_ERR_INVALID_ARG, "bad rank / nranks");
  ncclUniqueId id;
  std::memcpy(&id, uid, sizeof id);
  ncclComm_t c;
  ncclResult_t r = ncclCommInitRank(&c, nranks, id, rank);
  if (r != ncclSuccess) return fail(PERF_ERR_NCCL, ncclGetErrorString(r));
  if (p->comm) ncclCommDestroy(p->comm);
  p->comm = c;
  p->rank = rank;
  p->nranks = nranks;
  // connect the ring neighbours now (a 4-byte exchange), not lazily inside the
  // first (possibly graph-captured) halo exchange
  if (nranks > 1) {
    void* d = nullptr;
    cudaStream_t ws = nullptr;
    CK(cudaMalloc(&d, 16));
    CK(cudaStreamCreateWithFlags(&ws, cudaStreamNonBlocking));
    char* b = static_cast<char*>(d);
    ncclGroupStart();
    if (rank > 0) {
      ncclSend(b, 4, ncclUint8, rank - 1, c, ws);
      ncclRecv(b + 4, 4, ncclUint8, rank - 1, c, ws);
    }
    if (rank < nranks - 1) {
      ncclSend(b + 8, 4, ncclUint8, rank + 1, c, ws);
      ncclRecv(b + 12, 4, ncclUint8, rank + 1, c, ws);
    }
    ncclResult_t rr = ncclGroupEnd();
    cudaError_t e = cudaStreamSynchronize(ws);
    cudaStreamDestroy(ws);
    cudaFree(d);
    if (rr != ncclSuccess) return fail(PERF_ERR_NCCL, std::string("neighbour warm-up: ") + ncclGetErrorString(rr));
    if (e != cudaSuccess) return cuda_fail(e, "neighbour warm-up");
  }
  return PERF_OK;
}

// ------------------------------------------------------- NEXT-4 peer links ----
namespace {
struct P2PBlob {  // what perf_p2p_export writes (PERF_P2P_HANDLE_BYTES = 128)
  uint32_t magic, W, H, hb;
  int32_t band_y0, pad[3];
  cudaIpcMemHandle_t handle;  // 64 bytes
};
static_assert(sizeof(P2PBlob) <= 128, "blob size");
constexpr uint32_t kP2PMagic = 0x4B503250u;  // "P2PK"
}  // namespace

perf_status perf_p2p_export(perf_plan_t p, void* out) {
  if (!p || !out) return fail(PERF_ERR_INVALID_ARG, "NULL argument");
  if (p->app != PERF_APP_HOTSPOT) return fail(PERF_ERR_INVALID_ARG, "P2P halos are for banded Hotspot plans");
  perf_status st = band_alloc(p);
  if (st != PERF_OK) return st;
  P2PBlob b;
  std::memset(&b, 0, sizeof b);
  b.magic = kP2PMagic;
  b.W = (uint32_t)p->W;
  b.H = (uint32_t)p->H;
  b.hb = (uint32_t)p->band.hb;
  b.band_y0 = (int32_t)p->band_y0;
  CK(cudaIpcGetMemHandle(&b.handle, p->band.base));
  std::memset(out, 0, PERF_P2P_HANDLE_BYTES);
  std::memcpy(out, &b, sizeof b);
  return PERF_OK;
}

perf_status perf_p2p_attach(perf_plan_t p, const void* up, const void* down) {
  if (!p) return fail(PERF_ERR_INVALID_ARG, "NULL plan");
  perf_status st = band_alloc(p);
  if (st != PERF_OK) return st;
  Band& B = p->band;
  const void* blobs[2] = {up, down};
  for (int k = 0; k < 2; ++k) {
    if (!blobs[k]) continue;
    P2PBlob b;
    std::memcpy(&b, blobs[k], sizeof b);
    if (b.magic != kP2PMagic || (int)b.W != p->W || (int)b.hb != B.hb)
      return fail(PERF_ERR_INVALID_ARG, "peer handle: not a band of this grid (W / halo mismatch)");
    const long long adj = k == 0 ? (long long)b.band_y0 + b.H : (long long)p->band_y0 + p->H;
    if (adj != (k == 0 ? p->band_y0 : (long long)b.band_y0))
      return fail(PERF_ERR_INVALID_ARG, "peer handle: band is not adjacent");
    void* m = nullptr;
    CK(cudaIpcOpenMemHandle(&m, b.handle, cudaIpcMemLazyEnablePeerAccess));
    const BandLayout L = band_layout((size_t)b.H + 2 * b.hb, b.W);
    char* base = static_cast<char*>(m);
    B.peer_ipc[k] = m;
    B.peer_buf[k][0] = reinterpret_cast<float*>(base);
    B.peer_buf[k][1] = reinterpret_cast<float*>(base + L.arr);
    B.peer_pbuf[k] = reinterpret_cast<float*>(base + 2 * L.arr);
    // my slot in the neighbour's flags: the upper band reads "from lower" (1), the lower "from upper" (0)
    B.peer_flag[k] = reinterpret_cast<unsigned*>(base + 3 * L.arr) + (k == 0 ? 1 : 0);
    B.peer_row0[k] = b.band_y0 - (int)b.hb;
  }
  B.p2p = true;
  return PERF_OK;
}

perf_status perf_destroy(perf_plan_t p) {
  if (!p) return PERF_OK;
  if (p->d_err) cudaFree(p->d_err);
  if (p->d_tmp) cudaFree(p->d_tmp);
  if (p->d_stage_in) cudaFree(p->d_stage_in);
  if (p->d_stage_out) cudaFree(p->d_stage_out);
  host_pipe_free(p);
  hotspot_graph_free(p);
  if (p->s_cap) cudaStreamDestroy(p->s_cap);
  if (p->s_x) cudaStreamDestroy(p->s_x);
  if (p->ev_b) cudaEventDestroy(p->ev_b);
  if (p->ev_x) cudaEventDestroy(p->ev_x);
  band_free(p);
  if (p->comm) ncclCommDestroy(p->comm);
  delete p;
  return PERF_OK;
}

}  // extern "C"

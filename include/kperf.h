/*
 * kperf.h -- C ABI of the B200-native hot path of local memory-aware kernel
 * perforation (Maier, Cosenza, Juurlink, CGO'18; PAPER.md = the paper text).
 *
 * The paper states the problem as "input buffer -> data perforation -> data
 * reconstruction -> kernel execution -> output buffer" (Fig. 1b,
 * PAPER.md:258-274) with the perforation scheme, the reconstruction technique,
 * the perforation rate and the work-group size as parameters (Sec. 6.3,
 * PAPER.md:808-852).  Every entry point below is extern "C", takes plain
 * pointers and sizes, returns a perf_status (PERF_OK = 0) and never throws.
 * On failure perf_last_error() returns a thread-local message.
 *
 * Data layout: row-major, dense, pitch = W * sizeof(T); a batch of BATCH
 * frames is frame-major (frame f starts at element f * W * H).  T is uint8_t
 * for PERF_APP_MEDIAN and float for every other app.  Pixel (x, y) is element
 * y * W + x.
 *
 * Ownership: the caller owns every buffer it passes (device buffers for the
 * perf_run* calls, host buffers for perf_run_host) and keeps them alive until
 * the work on `stream` completes.  A plan owns only scratch (error partials,
 * Hotspot ping-pong/halo rows, staging buffers of perf_run_host).  `in` and
 * `out` must not alias.  A plan is used by one stream at a time.  `stream` is
 * a cudaStream_t (NULL = legacy default stream).
 *
 * Asynchrony: perf_run and perf_run_hotspot only enqueue work (asynchronous
 * faults surface at the next synchronising call); perf_error and
 * perf_run_host synchronise `stream` before returning.
 */
#ifndef KPERF_H
#define KPERF_H

#ifdef __cplusplus
extern "C" {
#endif

typedef enum {
  PERF_OK = 0,
  PERF_ERR_INVALID_ARG = 1, /* null pointer, bad size/enum/rate/radius, misuse */
  PERF_ERR_UNSUPPORTED = 2, /* a combination the build does not provide */
  PERF_ERR_CUDA = 3,        /* a CUDA runtime error (message in perf_last_error) */
  PERF_ERR_NCCL = 4,        /* an NCCL error (sharded Hotspot) */
  PERF_ERR_OOM = 5          /* scratch allocation failed */
} perf_status;

/* Applications of Sec. 6.1 (Table 1). */
typedef enum {
  PERF_APP_GAUSSIAN = 0,    /* binomial blur, radius 1 (3x3) or 2 (5x5), fp32 */
  PERF_APP_SOBEL = 1,       /* gradient magnitude, radius 1 (3x3) or 2 (5x5), fp32 */
  PERF_APP_MEDIAN = 2,      /* 3x3 median, radius 1, u8 */
  PERF_APP_HOTSPOT = 3,     /* Rodinia 2D thermal step, radius 1, fp32 (perf_run_hotspot) */
  PERF_APP_GAUSS_SOBEL = 4, /* Sobel3(Gaussian5(frame)), the C5 pipeline; radius must be 2 */
  PERF_APP_INVERSION = 5    /* 255 - x, radius 0, fp32 */
} perf_app;

/* Perforation schemes (Sec. 4.4; Fig. 4). */
typedef enum {
  PERF_SCHEME_NONE = 0,    /* exact kernel: every input element is loaded */
  PERF_SCHEME_ROW = 1,     /* skip whole rows; rebuilt along y */
  PERF_SCHEME_COL = 2,     /* skip G-pixel column granules; rebuilt along x */
  PERF_SCHEME_CHECKER = 3, /* skip G-pixel cells on a diagonal lattice; rebuilt along y */
  PERF_SCHEME_STENCIL1 = 4 /* the paper's Stencil1 (Sec. 4.4, Fig. 5): a work-group tile of
                              TILE1_W x TILE1_H outputs loads only its interior; its halo is
                              rebuilt by NN from the tile border.  rate must be {0, 1}.
                              Gaussian, Sobel, Median, Inversion. */
} perf_scheme;

/* Reconstruction techniques (Sec. 5.1). */
typedef enum {
  PERF_RECON_NN = 0,     /* nearest loaded element; equidistant -> lower coordinate */
  PERF_RECON_LINEAR = 1  /* linear interpolation; NN where one side is missing */
} perf_recon;

typedef enum {
  PERF_METRIC_MRE = 0,   /* mean over {e != 0} of |e - a| / |e| */
  PERF_METRIC_ME = 1,    /* sum |e - a| / sum |e|  (Sobel's "mean error", :580-584) */
  PERF_METRIC_MAE = 2    /* mean |e - a| */
} perf_metric;

/* Skipped fraction num/den of the scheme's lines (rows, column granules or
 * cells): num = 0 (exact), num = 1 (skip one line of every den: the line with
 * phase den-1) or num = den-1 (keep one line of every den: phase 0).
 * 1 <= den <= 8.  The paper's Rows1 = {1,2}, Rows2 = {3,4}. */
typedef struct { int num, den; } perf_rate;

typedef struct perf_plan_s* perf_plan_t;

/* perf_plan_set keys.  None of them changes results except GRANULE_BYTES
 * (the width G of a column/checker cell, part of the mask definition) and
 * METRIC. */
enum {
  PERF_KEY_BATCH = 1,          /* frames per perf_run (default 1) */
  PERF_KEY_ITERS = 2,          /* Hotspot steps per perf_run_hotspot (default 1) */
  PERF_KEY_GRANULE_BYTES = 3,  /* G * sizeof(T) for COL/CHECKER (default 128 = the measured B200 DRAM
                                  fill granule; smaller cells save no DRAM bytes; multiple of sizeof(T)) */
  PERF_KEY_GLOBAL_H = 4,       /* sharded Hotspot: rows of the whole grid (default H) */
  PERF_KEY_BAND_Y0 = 5,        /* sharded Hotspot: first global row of this rank's band (default 0) */
  PERF_KEY_TILE_W = 6,         /* consumer warps per CTA (1..8); tile width = warps * 32 * V */
  PERF_KEY_TILE_H = 7,         /* output rows per CTA segment (default 128) */
  PERF_KEY_METRIC = 8,         /* perf_metric used by perf_error (default: MRE; ME for Sobel apps) */
  PERF_KEY_LOADER = 9,         /* 0 auto, 1 TMA bulk rows, 2 cp.async 16 B, 3 scalar (any alignment),
                                  4 TMA bulk copies of kept cell runs (column / checker, <= 64 cells per tile
                                  row; never chosen by auto: 2.5x slower than 2 for 128-B cells) */
  PERF_KEY_RING = 10,          /* shared-memory ring depth in rows (0 = auto) */
  PERF_KEY_HALO_ROWS = 11,     /* read-only: rows a Hotspot band exchanges with each neighbour per step */
  PERF_KEY_TILE1_W = 12,       /* STENCIL1 tile width: power of two, 16..256 (fp32) / 16..512 (u8); default 16 */
  PERF_KEY_TILE1_H = 13,       /* STENCIL1 tile height, 1..1024; default 16 */
  PERF_KEY_PRODUCER = 14,      /* 0 auto = 1 dedicated producer warp; 2 bulk rows issued by consumer warp 0
                                  (only in builds with -DKPERF_IPROD=1; the default build ignores 2: the
                                  inline-producer code slowed every consumer loop) */
  PERF_KEY_TBLOCK = 15,        /* Hotspot temporal blocking: steps per launch, 1..8 (default 1).  CHANGES
                                  RESULTS: T is loaded (perforated, rebuilt) once per launch and the other
                                  steps of the launch read on-chip T (R19).
                                  NONE / ROW schemes; banded plans exchange TBLOCK + den halo rows per launch */
  PERF_KEY_P2P = 16,           /* perf_run_hotspot_bands_local only: 1 = halos by direct peer stores fused into
                                  the step kernels + epoch flags (the NEXT-4 path), 0 = device copies */
  PERF_KEY_CHK_COMPACT = 17,   /* read-only: 1 when perf_run (on aligned buffers) packs keep-one checkerboard
                                  ring slots with the row's kept cells only */
  PERF_KEY_OVERLAP = 18,       /* banded Hotspot (NCCL or bands_local): 1 (default) = each launch first computes
                                  the halo_rows boundary rows at both band edges, then exchanges them on a
                                  plan-owned stream while the interior rows compute; 0 = one
                                  whole-band launch, then the exchange.  Same results */
  PERF_KEY_GRAPH = 19,         /* perf_run_hotspot / bands_local: 1 (default) = the ITERS loop is captured once
                                  per (buffers, plan state) into a CUDA graph and replayed (one launch per
                                  call); 0 = eager launches.  Peer-store (P2P) plans always run eagerly.
                                  Reads 2 after a capture failed and the plan fell back to eager launches */
  PERF_KEY_EXCHANGE = 20,      /* MEASUREMENT ONLY: 0 skips every halo exchange of banded runs (results are
                                  then wrong at band edges) so the exchange's share of a step can be timed */
  PERF_KEY_FOLD = 21,          /* row scheme, fp32 Gaussian / Sobel / Gauss-Sobel, one kept row per period (den 2
                                  or keep-one den 4): 1 (default) = the rebuild is folded into the vertical pass
                                  -- per kept row one horizontal pass, each output row a compile-time weighted
                                  sum of kept rows; 0 = rebuild every row,
                                  then filter.  Same values (bit-identical on integer-valued inputs) */
  PERF_KEY_HOST_SKIP = 22,     /* perf_run_host, row scheme: 1 (default) = only the kept rows are copied host ->
                                  device (one strided 2-D copy per kept phase; the kernels never read a skipped
                                  row, so the perforation saves PCIe bytes as well as HBM bytes); 0 = whole
                                  frames.  Same results */
  PERF_KEY_H2D_BYTES = 23      /* read-only: bytes one perf_run_host call copies host -> device (BATCH frames) */
};

/* size of a perf_p2p_export handle */
#define PERF_P2P_HANDLE_BYTES 128

/* Create a plan.  Validates: W, H >= 1; radius allowed for the app (Gaussian,
 * Sobel {1,2}; Median, Hotspot {1}; Gauss-Sobel {2}; Inversion {0});
 * den in [1,8], num in {0, 1, den-1}; CHECKER needs H >= den (every column
 * must hold a loaded element).  No device work, no allocation on the device. */
perf_status perf_plan(perf_plan_t* plan, perf_app app, int W, int H, int radius, perf_scheme scheme,
                      perf_rate rate, perf_recon recon);
perf_status perf_plan_set(perf_plan_t plan, int key, long long value);
perf_status perf_plan_get(perf_plan_t plan, int key, long long* value);

/* Run the fused perforated load -> rebuild -> stencil kernel over BATCH frames
 * of device memory: in, out are device pointers to BATCH * W * H elements of T.
 * Asynchronous on `stream`. */
perf_status perf_run(perf_plan_t plan, const void* in, void* out, void* stream);

/* Same computation on HOST buffers (pinned or pageable): copies in -> device,
 * runs, copies out -> host, synchronises `stream`.  The plan owns the device
 * staging buffers. */
perf_status perf_run_host(perf_plan_t plan, const void* host_in, void* host_out, void* stream);
/* (Pipelined: the batch is cut into <= 16 row chunks; chunk i is copied in on a
 * plan-owned stream, the output rows it completes are computed on `stream`, and
 * copied out on a second plan-owned stream, so both PCIe directions and the
 * kernels overlap.  Host buffers should be pinned for the copies to overlap.
 * Row scheme: only the kept rows are copied in (PERF_KEY_HOST_SKIP); the
 * device staging copy of a skipped row is never read.) */

/* ITERS Hotspot steps on device buffers of W * H floats (a band of H rows
 * starting at global row BAND_Y0 of a GLOBAL_H-row grid when sharded).  T and
 * P are both perforated and rebuilt every step -- every TBLOCK-th step for T
 * when TBLOCK > 1 (one launch per TBLOCK steps, T kept in shared memory in
 * between; PERF_ERR_UNSUPPORTED for COL/CHECKER or banded plans).  temp_in is
 * not modified. */
perf_status perf_run_hotspot(perf_plan_t plan, const float* temp_in, const float* power, float* temp_out,
                             void* stream);

/* Single-device emulation of the sharded Hotspot (used by the tests): nb plans
 * describing consecutive bands of one grid (GLOBAL_H, BAND_Y0 set, same ITERS)
 * step in lockstep on `stream`; halo rows move by device copies instead of
 * NCCL, through the same band buffers and kernels as perf_run_hotspot.
 * temp_in, power, temp_out are whole-grid device buffers. */
perf_status perf_run_hotspot_bands_local(perf_plan_t* plans, int nb, const float* temp_in, const float* power,
                                         float* temp_out, void* stream);

/* Error of `approx` against `exact` (device pointers, BATCH * W * H elements of
 * the plan's T): the plan's metric in fp64, deterministic two-pass reduction.
 * Writes the value and the count of contributing elements; synchronises. */
perf_status perf_error(perf_plan_t plan, const void* exact, const void* approx, void* stream,
                       double* err_out, long long* count_out);

/* Deterministic partial sums of the error metric over BATCH * W * H elements
 * (device pointers): sums[0] = sum of the per-element terms (|e - a| / |e| over
 * e != 0 for MRE; |e - a| for ME / MAE), sums[1] = sum |e| (ME), sums[2] =
 * contributing element count (exact in fp64 below 2^53).  Sums of several
 * shards add elementwise; perf_error_finish turns them into the metric.
 * Synchronises `stream`.  (Table 1) */
perf_status perf_error_sums(perf_plan_t plan, const void* exact, const void* approx, void* stream, double sums[3]);
/* Host only (no device work): the plan's metric from (summed) partial sums:
 * MRE = sums[0] / sums[2], ME = sums[0] / sums[1], MAE = sums[0] / sums[2];
 * 0 when the denominator is 0. */
perf_status perf_error_finish(perf_plan_t plan, const double sums[3], double* err_out, long long* count_out);
/* Sharded error: every rank's perf_error_sums are summed
 * with ncclAllReduce(ncclFloat64, ncclSum) on the plan's communicator
 * (perf_comm_init), so every rank returns the metric of the whole sharded
 * batch.  Collective: every rank of the communicator calls it.  Without a
 * communicator it equals perf_error.  Synchronises `stream`. */
perf_status perf_error_allreduce(perf_plan_t plan, const void* exact, const void* approx, void* stream,
                                 double* err_out, long long* count_out);

/* Row-band partition: rank `rank` of `nranks` owns global rows
 * [BAND_Y0, BAND_Y0 + H) of a GLOBAL_H-row image or grid.  A band buffer holds
 * one frame as buf_rows = halo_rows + H + halo_rows rows of W elements; buffer
 * row i is global row BAND_Y0 - halo_rows + i (rows outside the image are
 * never read).  halo_rows = the rows an output row at a band edge can read
 * beyond the band: stencil radius (Hotspot: TBLOCK steps of radius 1; the
 * fused pipeline: 3) plus den for the row and checkerboard schemes (the
 * rebuild distance of a skipped row, R2).  Each exchange sends
 * buffer rows [send_up_row, + halo_rows) to up_rank, receives
 * [recv_up_row, + halo_rows) from it, and likewise with down_rank; a missing
 * neighbour (grid edge) is -1 and its rows are not exchanged.  Host only. */
typedef struct {
  int halo_rows, buf_rows;
  int up_rank, down_rank;
  int send_up_row, recv_up_row, send_down_row, recv_down_row;
} perf_halo_plan;
perf_status perf_band_halo(perf_plan_t plan, int rank, int nranks, perf_halo_plan* out);

/* One-shot row bands of a BATCH of images (SURVEY 8(e), C2/C3 sharded by rows):
 * `in_band` holds BATCH frames of perf_band_halo's buf_rows x W elements each
 * (frame f at f * buf_rows * W), the band's own rows at buffer rows
 * [halo_rows, halo_rows + H); `out` holds BATCH frames of H x W (the band's
 * output rows).  With a communicator (perf_comm_init) the halo rows of every
 * frame are first filled from the neighbouring ranks (one ncclGroup of
 * ncclSend / ncclRecv on `stream`; every rank calls it, collective); without
 * one the caller must have filled them.  The mask is anchored to global rows
 * (R2), so the bands' outputs equal the whole image's rows bit for
 * bit.  Asynchronous on `stream`.  PERF_ERR_UNSUPPORTED for Hotspot (use
 * perf_run_hotspot) and for STENCIL1 bands not starting on a tile row. */
perf_status perf_run_band(perf_plan_t plan, void* in_band, void* out, void* stream);

/* Attach an NCCL communicator built from a 128-byte ncclUniqueId (rank,
 * nranks) -- collective over the ranks.  Used by the sharded Hotspot (rank k
 * holds global rows [BAND_Y0, BAND_Y0 + H); neighbours exchange halo rows
 * every launch), perf_run_band and perf_error_allreduce.  The neighbour
 * connections are set up here (a tiny warm-up exchange), so later exchanges
 * can be captured into CUDA graphs. */
perf_status perf_comm_init(perf_plan_t plan, const void* nccl_unique_id, int rank, int nranks);
/* Fill a 128-byte buffer with a fresh ncclUniqueId (rank 0 calls this). */
perf_status perf_comm_unique_id(void* out_128_bytes);

/* NEXT-4: peer-memory halo exchange over NVLink / NVSwitch,
 * replacing NCCL for the banded Hotspot.  perf_p2p_export allocates this
 * band's buffers (band geometry: W, H, GLOBAL_H, BAND_Y0, scheme, TBLOCK must
 * be final) and writes PERF_P2P_HANDLE_BYTES describing them (a CUDA IPC
 * handle + geometry) for the neighbouring ranks.  perf_p2p_attach opens the
 * upper (rank - 1) and lower (rank + 1) bands' handles (NULL at the grid
 * edges) -- collective in the sense that every rank must attach before any
 * rank runs.  Afterwards perf_run_hotspot stores each launch's first / last
 * halo rows directly into the neighbours' buffers from inside the step
 * kernel and orders launches with epoch flags (fence.sc.sys + st.release.sys
 * / ld.acquire.sys polling); no NCCL call, no copy.  Every rank must run the
 * same number of perf_run_hotspot calls with the same ITERS / TBLOCK.  The
 * neighbours' processes must outlive the runs.  Errors: INVALID_ARG on a
 * handle of another grid or a non-adjacent band, CUDA on IPC failures. */
perf_status perf_p2p_export(perf_plan_t plan, void* handle_out);
perf_status perf_p2p_attach(perf_plan_t plan, const void* up_handle, const void* down_handle);

perf_status perf_destroy(perf_plan_t plan);
const char* perf_last_error(void);
const char* perf_version(void);

#ifdef __cplusplus
}
#endif
#endif /* KPERF_H */

// hotspot_tb.cuh -- launch interface of the temporally blocked Hotspot kernel
// (hotspot_tb.cu, R19).
#pragma once
#include <cuda_runtime.h>

namespace kp {

struct TBParams {
  const float* T;   // temperature; global row y at (y - in_row0) * W
  const float* P;   // power, same geometry
  float* out;       // output row y at (y - out_row0) * W
  int W, Hg;
  int in_row0, avail0, avail1, out_row0;  // rows [avail0, avail1) exist in T / P
  int y_begin, y_end;                     // output rows of this launch (global)
  int steps;                              // S
  int OW, OH, apron, pitch, tiles_x;
  int row_scheme, den, keep_one, li;      // row perforation (row_scheme = 0: exact)
  int vec;                                // 16-B loads allowed (W % 4 == 0, aligned buffers)
  float sdc, cx, cy, c0, pamb;             // sdc = step/Cap; cx = sdc/Rx, cy = sdc/Ry,
                                          // c0 = 1 - 2cx - 2cy - sdc/Rz, pamb = sdc amb / Rz (host, fp64 -> fp32)
  float* pu;                              // NEXT-4 peer halo stores (see KParams in engine.cuh)
  float* pd;
  int pu_row0, pd_row0, halo_rows;
};

// S = q.steps (1..8) steps on output rows [y_begin, y_end); fills the tile geometry
cudaError_t launch_hotspot_tb(TBParams q, cudaStream_t s);

}  // namespace kp

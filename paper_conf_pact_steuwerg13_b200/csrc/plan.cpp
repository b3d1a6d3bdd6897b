// plan.cpp — distribution planner (pure host arithmetic, no CUDA calls).
//
// P:L205-213 (Fig. 1): single = whole container on one GPU; copy = a full
// replica on each GPU; block = "each GPU stores a contiguous, disjoint chunk";
// overlap = the block chunk "together with one or several border elements of the
// neighboring chunk".  P:L214-222 (Fig. 2): for a matrix the unit is a row and
// "the overlap size specifies the number of rows at the borders of a chunk which
// are copied to the two neighboring GPUs".
// Readings: A1 chunk = ceil(units/G) (last parts short or empty); A2 matrices
// split by rows; A3 no halo storage beyond the container.
#include "skl_internal.h"

namespace skl {

Range block_range(size_t units, int G, int g) {
  const size_t chunk = (units + (size_t)G - 1) / (size_t)G;
  Range r{(size_t)g * chunk, (size_t)(g + 1) * chunk};
  if (r.lo > units) r.lo = units;
  if (r.hi > units) r.hi = units;
  return r;
}

Range core_range(size_t units, int G, const Dist& d, int g) {
  switch (d.kind) {
    case DSINGLE: return g == d.arg ? Range{0, units} : Range{0, 0};
    case DCOPY: return Range{0, units};
    case DBLOCK:
    case DOVERLAP: return block_range(units, G, g);
  }
  return Range{0, 0};
}

Range need_range(size_t units, int G, const Dist& d, int g) {
  Range r = core_range(units, G, d, g);
  if (d.kind != DOVERLAP || r.empty()) return r;
  const size_t h = (size_t)d.arg;
  r.lo = r.lo >= h ? r.lo - h : 0;
  r.hi = r.hi + h <= units ? r.hi + h : units;
  return r;
}

namespace {
// Owner of unit u in the source distribution (the device whose core holds it).
int owner(size_t units, int G, const Dist& from, size_t u) {
  switch (from.kind) {
    case DSINGLE: return from.arg;
    case DBLOCK:
    case DOVERLAP: {
      const size_t chunk = (units + (size_t)G - 1) / (size_t)G;
      return (int)(u / chunk);
    }
  }
  return -1;  // copy: never needed (every device holds everything)
}

void emit(std::vector<Transfer>& out, size_t units, int G, const Dist& from, int dst, size_t lo,
          size_t hi) {
  size_t u = lo;
  while (u < hi) {
    const int src = owner(units, G, from, u);
    size_t end = hi;
    if (from.kind == DBLOCK || from.kind == DOVERLAP) {
      const Range b = block_range(units, G, src);
      if (b.hi < end) end = b.hi;
    }
    out.push_back(Transfer{src, dst, u, u, end - u});
    u = end;
  }
}
}  // namespace

std::vector<Transfer> plan_transfers(size_t units, int G, const Dist& from, bool from_halo_valid,
                                     const Dist& to, bool to_halo) {
  std::vector<Transfer> out;
  if (from.kind == DNONE || to.kind == DNONE) return out;
  for (int g = 0; g < G; ++g) {
    const Range want = to_halo ? need_range(units, G, to, g) : core_range(units, G, to, g);
    if (want.empty()) continue;
    const Range have = from_halo_valid ? need_range(units, G, from, g) : core_range(units, G, from, g);
    if (have.empty()) {
      emit(out, units, G, from, g, want.lo, want.hi);
      continue;
    }
    // want \ have: at most two intervals, left then right (canonical order)
    if (want.lo < have.lo) emit(out, units, G, from, g, want.lo, std::min(want.hi, have.lo));
    if (want.hi > have.hi) emit(out, units, G, from, g, std::max(want.lo, have.hi), want.hi);
  }
  return out;
}

}  // namespace skl

// skl_internal.h — internal data model of libskl.so (not installed).
//
// Layers (SURVEY.md §1 "New build"): B1 device context (Ctx), B2 containers +
// coherence (Cont, Part), B3 distribution planner + redistribution (plan.cpp,
// container.cpp), B4 NVRTC customisation compiler (compiler.cpp), B5 skeleton
// executors (skeletons.cpp, kernels/*.cuh), B6 C ABI (capi.cpp, include/skl.h).
#pragma once

#include <cuda_runtime.h>
#include <nvtx3/nvToolsExt.h>

#include <atomic>
#include <cstdint>
#include <cstring>
#include <map>
#include <memory>
#include <mutex>
#include <set>
#include <stdexcept>
#include <string>
#include <vector>

#include "../../include/skl.h"

namespace skl {

// ------------------------------------------------------------------ errors
// NVTX ranges (SURVEY §5 tracing): one per skeleton call and redistribution,
// visible in nsys / ncu timelines; no-ops unless a tool is attached (NVTX v3 is
// header-only and loads the tool's injection library on first use).
struct NvtxRange {
  explicit NvtxRange(const char* name) { nvtxRangePushA(name); }
  ~NvtxRange() { nvtxRangePop(); }
  NvtxRange(const NvtxRange&) = delete;
  NvtxRange& operator=(const NvtxRange&) = delete;
};

struct Error : std::runtime_error {
  int code;
  Error(int c, const std::string& m) : std::runtime_error(m), code(c) {}
};
[[noreturn]] void fail(int code, const std::string& msg);
void cuda_check(cudaError_t e, const char* what);
#define SKL_CUDA(x) ::skl::cuda_check((x), #x)

// ------------------------------------------------------------------ types
struct TypeInfo {
  std::string name;  // C spelling used in generated source
  size_t size = 0, align = 1;
  std::string decl;  // struct declaration ("" for builtins)
};

// ------------------------------------------------------------------ distributions
enum DistKind { DNONE = SKL_DIST_NONE, DSINGLE = SKL_SINGLE, DCOPY = SKL_COPY,
                DBLOCK = SKL_BLOCK, DOVERLAP = SKL_OVERLAP };
struct Dist {
  int kind = DNONE;
  int arg = 0;  // device (single) or overlap size d (overlap)
  bool operator==(const Dist& o) const { return kind == o.kind && arg == o.arg; }
};
struct Range {
  size_t lo = 0, hi = 0;
  size_t size() const { return hi > lo ? hi - lo : 0; }
  bool empty() const { return hi <= lo; }
  bool contains(const Range& r) const { return r.empty() || (lo <= r.lo && r.hi <= hi); }
};
// plan.cpp — pure host arithmetic (readings A1-A3)
Range block_range(size_t units, int G, int g);
Range core_range(size_t units, int G, const Dist& d, int g);  // units device g owns/computes
Range need_range(size_t units, int G, const Dist& d, int g);   // units g stores (with halo)
struct Transfer {
  int src, dst;      // global devices
  size_t src_unit;   // first unit (global index) read from src's part
  size_t dst_unit;   // first unit (global index) written into dst's part
  size_t n;          // units
  int slot = 0;      // staging slot (combine gathers), else 0
};
// Transfers turning distribution `from` (all of its need ranges valid, or only
// core ranges when from_core_only) into `to` (need ranges incl. halo when
// to_halo).  Units already present on the destination device are not moved.
std::vector<Transfer> plan_transfers(size_t units, int G, const Dist& from, bool from_halo_valid,
                                     const Dist& to, bool to_halo);

// ------------------------------------------------------------------ compiler
// One NVRTC-compiled module per distinct source text.  A cudaLibrary is context
// independent, so one load serves every device.
struct Program {
  std::string source;
  std::vector<char> cubin;
  cudaLibrary_t lib = nullptr;
  std::map<std::string, cudaKernel_t> kernels;
  std::map<std::string, size_t> smem_set;  // dynamic smem attribute already raised
  std::map<std::string, int> occ;          // resident blocks/SM per (kernel, block, smem)
};

// ------------------------------------------------------------------ devices
struct Device {
  int global = 0;      // global device index g
  int phys = 0;        // CUDA ordinal
  cudaStream_t own = nullptr, stream = nullptr;  // library stream, current stream
  cudaEvent_t ev = nullptr;                      // scratch event for cross-stream sync
  int sm_count = 148;
  // copy-engine streams for chunked host<->device transfers that overlap with
  // kernels on `stream`, and a pool of reusable events
  cudaStream_t h2d = nullptr, d2h = nullptr;
  std::vector<cudaEvent_t> ev_pool;
};

struct Cont;
struct Skel;

struct Ctx {
  int G = 1;                   // global devices
  int first_local = 0, nlocal = 1;
  bool dist_mode = false;      // one process per GPU, NCCL between ranks
  bool offline = false;        // no devices: compile only (skl_init_offline)
  bool capturing = false;      // a CUDA graph capture is open on the device stream(s)
  cudaEvent_t cap_fork = nullptr;            // capture fork / join events (several devices)
  std::vector<cudaEvent_t> cap_join;
  int rank = 0, world = 1;
  void* nccl_comm = nullptr;   // ncclComm_t
  void* shm_comm = nullptr;    // host shared-memory loopback transport (SKL_COMM=shm, tests)
  void* ipc = nullptr;         // IPC heap + peer mappings + barriers (SKL_COMM=ipc, ipc.cpp)
  std::vector<Device> dev;     // local devices, index g - first_local
  std::vector<TypeInfo> types; // index = skl_type (builtins first)
  std::set<Cont*> conts;
  std::set<Skel*> skels;
  // options
  int block_threads = 256;
  int debug_bounds = 0;
  int map_unroll = 4;
  int scan_chunks = 8;         // 16-byte chunks per thread in a Scan tile
  int scan_persistent = 1;     // (unused since the chunked Scan; kept for the option API)
  int scan_sub = 4;            // Scan tiles per look-back chunk
  int scan_fstride = 16;       // Scan status word spacing (8-byte units; 16 = one L2 line)
  int scan_spin_ns = 0;        // Scan look-back spin back-off (__nanosleep)
  int scan_minb = 5;           // Scan per-tile kernels: min resident blocks (launch bounds)
  int scan_minb_pipe = 2;      // Scan pipelined kernel: min resident blocks
  int scan_lbw = 1;            // Scan look-back: predecessors watched per thread (2-6 measured slower)
  int mo_rh = 0, mo_cw = 0;    // MapOverlap outputs per thread (rows x cols); 0 = auto
  int mo_minb = 0;             // MapOverlap min resident blocks per SM (0 = 64-register cap)
  int mo_persist = 0;          // MapOverlap 2-D: persistent blocks, double-buffered tiles
  int mo_tma = 1;              // MapOverlap 2-D: one TMA copy stages a block's tile (skl_mo2d_t)
  int mo_kt = 0;               //   tiles per block (stacked vertically, copies issued up front; 0 = auto)
  int mo_full = -1;            //   unguarded full-tile apply loop (-1 = auto: with 2+ tiles per block)
  int mo_ws = 0;               // MapOverlap 2-D: TMA producer warp + consumer warps (skl_mo2d_ws)
  int mo_ws_stages = 4;        //   shared-memory ring depth
  int mo_ws_minb = 0;          //   resident blocks per SM the registers must allow (0 = auto)
  int lazy_fusion = 1;         // defer Zip/Map without an output (fused into a Reduce)
  int halo_push = 1;           // MapOverlap stores its border rows into the neighbours' halos
  int map_interleave = 0;      // Map/Zip: warp-interleaved elements (divergent functions)
  int map_il_elems = 0;        //   elements per lane of the interleaved kernel (0 = one chunk)
  int map_auto = 1;            //   functions with a loop: interleaved, one element per lane
  int xfer_kernel = 1;         // one process: redistribution moves as one batched kernel per device
  int combine_unroll = 0;      // copy(+) -> block folds: 16-byte chunks per thread (0 = 2)
  int combine_peer = 1;        // one process: copy(+) -> block folds straight from the peers' replicas
                               // (0 = staged exchange then fold, 2 = one kernel per device even on one GPU)
  int xfer_chunks = 8;         // host<->device transfers split into this many chunks per part
  int xfer_taper = 1;          //   the last two chunks 1/2 and 1/4 of the others (short tail)
  int ap_fast = 1;             // Allpairs zip-reduce: 128-row tiles (4-byte inputs, d % 4 == 0)
  int ap_tile = 0;             // Allpairs tile columns: 0 = by wave fill, 8 = 128, 4 = 64, 2 = hybrid
  int ap_bk = 0;               // Allpairs 128-row kernels: k-slice depth (0 = 16)
  int ap_hybrid = 1;           // Allpairs: last partial wave of 128 x 128 tiles as 128 x 64 halves
  std::vector<std::vector<char>> peer_ok;  // [g][h]: device g can store to device h's memory
  // Scan schedule: 6 = one block per tile, tile kept in shared memory, low
  // register count so 5 tiles fit per SM (default, fastest measured: 5.8 TB/s
  // on 2^30 int32); 3 = one block per tile, items in registers, block-wide
  // look-back; 2 = as 3 with a warp-wide look-back; 4 = persistent 3-stage
  // pipeline; 0 = persistent chunked (L2 re-read); 1 / 5 / 7 = measurement
  // only: 3 / 4 / 6 without look-back (wrong results, the pipeline's ceiling)
  int scan_variant = 6;
  // counters
  std::atomic<long long> n_launch{0}, n_compile{0}, n_cache_hit{0}, h2d{0}, d2h{0}, p2p{0}, pushed{0}, n_disk_hit{0}, n_tma{0}, n_nccl_group{0};
  int composed_id = 0;  // names of composed Map chains (lazy fusion)
  // optional caller-provided device allocator (skl_set_allocator)
  void* (*user_alloc)(size_t, int, void*, void*) = nullptr;
  void (*user_free)(void*, int, void*, void*) = nullptr;
  void* alloc_user = nullptr;
  // NVRTC cache: source hash -> program
  std::map<std::string, std::unique_ptr<Program>> programs;
  // builtin kernels (fill) per element size
  bool is_local(int g) const { return g >= first_local && g < first_local + nlocal; }
  Device& D(int g) { return dev.at((size_t)(g - first_local)); }
  const TypeInfo& type(int t) const;
  void set_device(int g);
};

// ------------------------------------------------------------------ containers
// A unit range of a part that becomes valid when `ev` completes (chunked
// upload on the copy stream, or a chunk of a Map's output); consumers on the
// device stream wait for it, or stream it out chunk by chunk.
struct Ready {
  Range r;
  cudaEvent_t ev = nullptr;
};
struct Part {
  void* ptr = nullptr;  // device buffer; addresses unit buf.lo
  Range buf;            // units the buffer covers
  Range valid;          // units holding valid data (subset of buf)
  size_t cap_bytes = 0;
  std::vector<Ready> ready;  // pending chunks (empty: everything is ordered on the stream)
};

// A Zip/Map called without an output container is deferred (lazy fusion,
// SURVEY §8(f)1): a Reduce that consumes it computes the elements on the fly;
// any other use, or a write to an input, materialises it first.
struct Lazy {
  Skel* s = nullptr;  // the deferred Zip/Map (nullptr: not lazy)
  Cont* l = nullptr;
  Cont* r = nullptr;  // Zip's right input
  Dist d;             // distribution the elements are computed in
};

struct Cont {
  Ctx* ctx = nullptr;
  Lazy lazy;
  std::vector<Cont*> dependents;  // lazy containers that read this one
  int type = 0;
  size_t elt = 0;          // element bytes
  bool matrix = false;
  size_t rows = 0, cols = 1;  // vector: rows = n, cols = 1
  size_t units() const { return rows; }
  size_t unit_bytes() const { return cols * elt; }
  size_t bytes() const { return rows * cols * elt; }
  Dist dist;
  bool dev_valid = false;    // core ranges of `dist` valid on every device
  bool halo_valid = false;   // overlap halos valid too
  bool diverged = false;     // copy replicas written independently
  Skel* combine = nullptr;   // copy(+) combine function (A25)
  std::vector<void*> stage;  // combine staging per device (kept for the next combine)
  std::vector<size_t> stage_bytes;
  std::vector<Part> parts;   // indexed by global device; only local ones used
  void* host = nullptr;      // pinned host mirror (lazily allocated)
  bool host_valid = false;
  size_t spare_halo = 0;     // allocate parts with this many extra halo units
  // block-distributed, but the buffers already hold valid halos of this many
  // units (pushed by the producing MapOverlap): overlap(d <= halo_ready) is free
  size_t halo_ready = 0;
};

// container.cpp
Cont* cont_create(Ctx* ctx, int type, size_t rows, size_t cols, bool matrix);
void cont_destroy(Cont* c);
// Make `c` hold valid data in distribution `d` on the devices (upload from the
// host mirror or redistribute device-to-device as needed).  `halo` = overlap
// halos must be valid too.
// keep_ready: leave chunk events of an upload pending for the caller (a Map/Zip
// consumes the chunks as they arrive); otherwise every pending chunk is ordered
// before later work on the device stream.
void ensure(Cont* c, const Dist& d, bool halo, bool keep_ready = false);
void sync_ready(Cont* c);  // device streams wait for every pending chunk of c
// Prepare `c` as an output in distribution `d` (contents will be overwritten on
// the core ranges); allocates parts with `spare` halo units of room.
void prepare_output(Cont* c, const Dist& d, size_t spare);
void mark_written(Cont* c);  // devices valid, host stale, halos stale
void* part_ptr(Cont* c, int g, size_t unit);  // device pointer to global unit on device g
void host_upload(Cont* c, const void* host);  // into current distribution
void host_download(Cont* c, void* host);      // whole container (collective)
void download_part(Cont* c, int g, void* host, size_t* first, size_t* n);
void fill(Cont* c, const void* value);
void* host_mirror(Cont* c, int mode);
void copy_combine_to_copy(Cont* c);  // fold diverged replicas, keep copy
// lazy fusion (skeletons.cpp)
void materialize(Cont* c);             // run c's deferred Zip/Map, if any
void materialize_dependents(Cont* c);  // before c's values change
void drop_lazy(Cont* c);               // c is overwritten or destroyed

// comm.cpp — execute transfers between per-device buffers.  srcp/dstp resolve
// (device, unit) to a device pointer for LOCAL devices.
struct PtrFn {
  virtual void* src(const Transfer& t) = 0;  // local t.src only
  virtual void* dst(const Transfer& t) = 0;  // local t.dst only
  virtual ~PtrFn() = default;
};
void run_transfers(Ctx* ctx, const std::vector<Transfer>& tr, size_t unit_bytes, PtrFn& p);
// one batched copy launch on device g's stream (builtin.cu); sources are on
// g's GPU or a peer with access enabled
constexpr int kXferMaxSegs = 32;
// threads per block of the peer folds (skl_combine_peer / skl_combine_all); the
// Reduce/Scan programs are compiled with SKL_CBLOCK set to this value
constexpr int kCombineBlock = 256;
struct XferSeg {
  const void* src;
  void* dst;
  size_t bytes;
};
void launch_xfer_batch(Ctx* ctx, int g, const std::vector<XferSeg>& segs);
void barrier_streams(Ctx* ctx);  // every local stream waits for every other
cudaEvent_t event_get(Ctx* ctx, int g);
void event_put(Ctx* ctx, int g, cudaEvent_t e);
// one process per GPU over NVLink peer memory (ipc.cpp, SKL_COMM=ipc)
constexpr int kIpcMaxRanks = 8;
bool ipc_requested();
void ipc_init(Ctx* ctx, const void* id128);
void ipc_destroy(Ctx* ctx);
void* ipc_alloc(Ctx* ctx, size_t bytes);
void ipc_free(Ctx* ctx, void* ptr);
// collective: every rank passes its values, gets every rank's (host barrier)
std::vector<std::vector<uint64_t>> ipc_exchange(Ctx* ctx, const std::vector<uint64_t>& mine);
void* ipc_translate(Ctx* ctx, int rank, uint64_t va);  // rank's device address, mapped here
void ipc_barrier(Ctx* ctx);  // device barrier of every rank's stream (collective)
void ipc_check(Ctx* ctx);
// NCCL (dlopen)
void nccl_get_unique_id(void* out128);
void nccl_init(Ctx* ctx, const void* id);
void nccl_destroy(Ctx* ctx);

// ------------------------------------------------------------------ compiler.cpp
std::string program_source(Ctx* ctx, const std::string& body);
Program* compile(Ctx* ctx, const std::string& source, std::string* log_out);
void launch(Ctx* ctx, int g, Program* prog, const char* kernel, dim3 grid, dim3 block,
            size_t smem, void** args);
int max_smem_optin(Ctx* ctx, int g);
int occupancy(Ctx* ctx, int g, Program* prog, const char* kernel, int block, size_t smem);
std::string detect_entry(const std::string& src);
bool has_loop(const std::string& src);
std::string kernel_template(const char* name);  // embedded kernels/*.cuh

// ------------------------------------------------------------------ skeletons
enum SkelKind { K_MAP = 1, K_ZIP, K_REDUCE, K_SCAN, K_MAPOVERLAP, K_ALLPAIRS };
struct Scratch {  // per-device persistent scratch (reduce partials, scan status)
  void* ptr = nullptr;
  size_t bytes = 0;
};
struct Skel {
  Ctx* ctx = nullptr;
  int kind = 0;
  std::string user_src, entry;
  int tin = 0, tin2 = 0, tout = 0;
  std::vector<int> extra;  // extra arg types (with SKL_PTR flag)
  int d = 0, boundary = 0;
  std::vector<unsigned char> neutral;
  Program* prog = nullptr;
  Program* prog1d = nullptr;        // MapOverlap on vectors (compiled lazily)
  std::map<int, Scratch> scratch_red;    // per device: reduce ticket counter + block partials
  std::map<int, Scratch> scratch_scan;   // per device: decoupled look-back status
  std::map<int, Scratch> scratch_stage;  // per device: cross-device partials / totals
  std::map<int, uint32_t> epoch;    // scan lookback epochs per device
  // MapOverlap tile geometry (compile-time constants of prog)
  int mo_tw = 0, mo_th = 0, mo_pitch = 0, mo_a = 0, mo_rh = 0, mo_cw = 0;
  int mo_kt = 1;            // TMA tile kernel: tiles per block (SKL_MO_KT)
  bool mo_auto_rh = false;  // byte images: row count chosen after compiling (spill check)
  bool mo_auto_byte = false;  // byte images, geometry automatic: 8 x 8 block for heavy functions
  std::string mo_defs;      // program defines without the row count
  bool mo_1d = false;
  int scan_ch = 0;   // Scan: 16-byte chunks per thread (0 = generic path)
  int cunr = 2;      // Reduce/Scan programs: 16-byte chunks per thread of the copy(+) folds (SKL_CUNR)
  int scan_sub = 4;  // Scan: tiles per look-back chunk (vector path)
  int scan_variant = 0;
  int scan_fstride = 16;  // Scan: status word spacing in 8-byte units
  int bounds = 0;         // MapOverlap: 1 = get() offsets statically proven within d
  bool ap_zr = false;     // Allpairs: zip-reduce form
  int block = 256;   // threads per block the program was compiled for
  int unroll = 4;    // Map/Zip chunks per thread the program was compiled for
  int ilj = 4;       // Map/Zip interleaved kernel: elements per lane (SKL_ILJ)
  bool interleave = false;  // Map/Zip: launch the warp-interleaved kernel
  std::map<Skel*, Program*> fused;  // Reduce: fused programs per producing Zip/Map
  std::map<Skel*, Skel*> composed;  // Map g: g∘f per producing Zip/Map f (nullptr: not composable)
};
Skel* skel_create(Ctx* ctx, int kind, const char* src, const char* entry, int tin, int tin2,
                  int tout, const int* extra, int nextra, int d, int boundary, const void* neutral);
void skel_destroy(Skel* s);
void run_map(Skel* s, Cont* in, Cont** out, const skl_arg* extra, int nextra);
void run_zip(Skel* s, Cont* l, Cont* r, Cont** out, const skl_arg* extra, int nextra);
void run_reduce(Skel* s, Cont* in, Cont** out);
void run_scan(Skel* s, Cont* in, Cont** out);
void run_mapoverlap(Skel* s, Cont* in, Cont** out);
Skel* allpairs_create(Ctx* ctx, const char* src, const char* entry, const char* rsrc,
                      const char* rentry, int tin, int tout);  // rsrc != NULL: zip-reduce form
void run_allpairs(Skel* s, Cont* a, Cont* b, Cont** out);
// ordered combine of G staged replica slices into dst (A25), on device g
void run_combine(Skel* s, int g, const void* staging, size_t stride_elems, int nrep, void* dst,
                 size_t nelem);
void run_combine_peer(Skel* s, int g, const void* const* srcs, int nrep, void* dst, size_t nelem);
void run_combine_all(Skel* s, int g, const void* const* bases, int nrep, size_t nelem, size_t chunk_elems);
void* device_alloc(Ctx* ctx, int g, size_t bytes);
void device_free(Ctx* ctx, int g, void* p);
void check_debug_flag(Ctx* ctx);
// bounds.cpp: 1 proven, 0 unknown, -1 violation (reason in *why)
int check_get_bounds(const std::string& src, int d, std::string* why);

}  // namespace skl

// C handles (include/skl.h) wrap the internal objects.
struct skl_ctx { skl::Ctx* c; };
struct skl_cont { skl::Cont* c; };
struct skl_skel { skl::Skel* s; };

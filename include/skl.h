/*
 * skl.h — C ABI of libskl.so, a B200-native (sm_100a) implementation of the
 * data-parallel hot path of SkelCL (Steuwer & Gorlatch, "SkelCL: Enhancing
 * OpenCL for High-Level Programming of Multi-GPU Systems", PaCT 2013;
 * /root/reference/PAPER.md, cited as P:Lx-y).  Readings of passages the paper
 * leaves open are numbered A<n> and listed in DESIGN.md §3.
 *
 * Conventions:
 *  - Every call returns skl_status: SKL_OK (0) or a negative SKL_ERR_* code.
 *    skl_last_error() returns a thread-local message (with the NVRTC log for
 *    SKL_ERR_COMPILE).  Nothing here aborts the process.
 *  - Handles are opaque and owned by the library.  The caller destroys
 *    containers and skeletons; skl_finalize() frees everything still alive.
 *  - A context is driven by one host thread, matching the paper's sequential
 *    host program.
 *  - Calls enqueue asynchronously on one stream per device.  Only calls that
 *    hand data to the host (skl_copy_out, skl_host_data, skl_scalar_get,
 *    skl_sync) wait.
 *  - Pointers named `host` are host memory (pinned memory gives DMA speed);
 *    pointers returned by skl_local_part are device memory, borrowed.
 *  - There is no CPU fallback: every skeleton runs as CUDA kernels for
 *    sm_100a, JIT-compiled with NVRTC from the user's source string.  Without a
 *    usable GPU, skl_init returns SKL_ERR_CUDA.
 */
#ifndef SKL_H
#define SKL_H
#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef int skl_status;
#define SKL_OK 0
#define SKL_ERR_INVALID_ARG -1   /* bad handle, NULL pointer, bad enum value      */
#define SKL_ERR_TYPE -2          /* element types do not fit the skeleton         */
#define SKL_ERR_SIZE_MISMATCH -3 /* Zip inputs of different sizes    */
#define SKL_ERR_EMPTY -4         /* Reduce / Scan of an empty vector (A11)        */
#define SKL_ERR_COMPILE -5       /* NVRTC rejected the source; log in last_error  */
#define SKL_ERR_OUT_OF_RANGE -6  /* debug bounds: get() beyond d (A21) */
#define SKL_ERR_DISTRIBUTION -7  /* distribution request that cannot be honoured  */
#define SKL_ERR_OOM -8           /* device or pinned-host allocation failed       */
#define SKL_ERR_CUDA -9          /* CUDA runtime error (message in last_error)    */
#define SKL_ERR_NCCL -10         /* NCCL error in multi-process mode              */
#define SKL_ERR_UNSUPPORTED -11  /* feature not available (e.g. NCCL library)    */

typedef struct skl_ctx skl_ctx;
typedef struct skl_cont skl_cont;
typedef struct skl_skel skl_skel;

/* ------------------------------------------------------------------ types
 * Element types of containers and of customising-function parameters.  The
 * paper's examples use int, float, char and complex numbers (P:L156, P:L254,
 * P:L468).  Struct element types (A27, LM OSEM events) are registered
 * with skl_type_struct.  OR-ing SKL_PTR into an *extra-argument* type declares a
 * container argument (the customising function receives `T*`).               */
typedef int skl_type;
#define SKL_VOID 0
#define SKL_U8 1   /* uchar / unsigned char                                   */
#define SKL_I8 2
#define SKL_I32 3  /* int                                                     */
#define SKL_U32 4  /* uint                                                    */
#define SKL_F32 5  /* float                                                   */
#define SKL_F64 6  /* double                                                  */
#define SKL_F32X2 7 /* float2 (complex numbers, Mandelbrot P:L468)            */
#define SKL_I64 8
#define SKL_U64 9
#define SKL_I16 10
#define SKL_U16 11
#define SKL_PTR 0x1000
/* Register a struct type.  `name` is the C identifier used in sources,
 * `decl_src` its definition (e.g. "struct Event { float x0,y0,z0,x1,y1,z1; };"),
 * size/align as the C compiler lays it out.  The declaration is prepended to
 * every program that uses the type.  Returns the new type id in *out.          */
skl_status skl_type_struct(skl_ctx* ctx, const char* name, const char* decl_src, size_t size,
                           size_t align, skl_type* out);
skl_status skl_type_size(skl_ctx* ctx, skl_type t, size_t* size);

/* ------------------------------------------------------------------ context
 * SkelCL::init(): "the calculation specified by a skeleton is
 * performed automatically on all GPUs available".
 *
 * skl_init: one process drives `ndev` devices.  devices[g] is the CUDA ordinal
 * of logical device g; NULL means all visible GPUs (ndev = 0) or devices
 * g % visible (ndev > 0).  Several logical devices may share one physical GPU
 * ("logical-device mode"): each gets its own stream and its own
 * memory, and data moves between them by device-to-device copies, so the whole
 * distribution machinery runs on a 1-GPU box.
 *
 * skl_init_dist: one process per GPU (torchrun).  Global device g is rank g;
 * `nccl_id` is the 128-byte id from skl_nccl_unique_id() on rank 0, broadcast
 * by the caller.  The transport between the ranks is chosen by the environment
 * variable SKL_COMM (identical on every rank):
 *   "ipc" (default; the ranks of one node): device memory comes from an IPC
 *     heap, each rank maps the peers' buffers with CUDA IPC, and every exchange
 *     (redistribution, halo push, copy(+) fold, Reduce partials, Scan carries)
 *     runs as in-kernel peer loads/stores ordered by device barriers; the id is
 *     the name of a POSIX shared-memory control block; a barrier that waits
 *     more than 60 s fails the next call with SKL_ERR_NCCL instead of hanging;
 *   "nccl": NCCL send/recv of the same transfer lists (libnccl.so.2 - the copy
 *     already loaded in the process, if any - is loaded on first use; the id is
 *     an ncclUniqueId);
 *   "shm": a host shared-memory loopback (tests, several ranks on one GPU).
 * With world == 1 the context is the one-process form unless SKL_DIST_FORCE=1,
 * which keeps the multi-process code path and sets up the transport anyway
 * (tests: NCCL's communicator setup, group calls and teardown on one GPU).
 * Every rank must issue the same sequence of calls (SPMD): host-visible results
 * and redistributions are collective.                                          */
skl_status skl_init(int ndev, const int* devices, skl_ctx** out);
skl_status skl_init_dist(int rank, int world, int cuda_device, const void* nccl_id, skl_ctx** out);
skl_status skl_nccl_unique_id(void* out128);
skl_status skl_finalize(skl_ctx* ctx);
skl_status skl_num_devices(skl_ctx* ctx, int* ndev, int* first_local, int* nlocal);
/* Use the caller's stream (e.g. torch's current stream) for device g; NULL
 * restores the library's own stream.  Only local devices.                      */
skl_status skl_set_stream(skl_ctx* ctx, int g, void* cuda_stream);
skl_status skl_get_stream(skl_ctx* ctx, int g, void** cuda_stream);
skl_status skl_sync(skl_ctx* ctx);
/* Device memory from the caller's allocator instead of the library's
 * cudaMallocAsync pool (e.g. torch's caching allocator, so that
 * PyTorch owns device memory).  alloc(bytes, cuda_device, cuda_stream, user)
 * returns a device pointer usable in stream order on cuda_stream (NULL ->
 * SKL_ERR_OOM); release(ptr, cuda_device, cuda_stream, user) returns it.  Every
 * container part and skeleton scratch buffer goes through them.  Only before
 * any container or skeleton exists (else SKL_ERR_INVALID_ARG); both NULL
 * restores the default.                                                        */
typedef void* (*skl_alloc_fn)(size_t bytes, int cuda_device, void* cuda_stream, void* user);
typedef void (*skl_free_fn)(void* ptr, int cuda_device, void* cuda_stream, void* user);
/* (With the "ipc" transport of skl_init_dist every buffer comes from the IPC
 * heap, which peers must be able to map; a caller's allocator is not used.)    */
skl_status skl_set_allocator(skl_ctx* ctx, skl_alloc_fn alloc, skl_free_fn release, void* user);
/* Options: "block_threads" (work-group size; default 256),
 * "debug_bounds" (1 = get() range-checked, A21), "map_unroll" (chunks per
 * thread, default 4), "lazy_fusion" (1 = a Map/Zip without an output is
 * deferred and fused into the Reduce that consumes it; default 1),
 * "halo_push" (1 = a MapOverlap on several devices of this process stores its
 * border units into the neighbours' halo units, so the next overlap read
 * exchanges nothing; default 1), "map_interleave" (1 = lane l of a
 * warp handles elements base + 32 j + l: for customising functions whose cost
 * varies per element, e.g. Mandelbrot; default 0), "map_il_elems" (elements
 * per lane of the interleaved kernel; 0 = one 16-byte chunk's worth; default 0),
 * "map_auto" (1 = a Map/Zip whose customising source holds a loop - for /
 * while / do - uses the interleaved kernel with one element per lane unless
 * map_interleave / map_il_elems say otherwise; default 1),
 * "ap_fast" (Allpairs
 * zip-reduce 128 x 128 tiles for 4-byte inputs with d % 4 == 0; default 1),
 * "ap_hybrid" (1 = when the 128 x 128 tiles leave the last wave less than half
 * full, that wave runs as 128 x 64 halves; default 1), "ap_tile" (0 = automatic,
 * 8 / 4 = force 128 / 64 tile columns, 2 = force the hybrid),
 * "xfer_kernel" (1 = with several devices in this process, the moves of a
 * redistribution or halo refresh into one GPU run as one batched copy kernel
 * (peer loads over NVLink between GPUs); 0 = one cudaMemcpy(Peer)Async per
 * move; default 1), "xfer_chunks" (host <-> device transfers of >= 4 MB per
 * part go in this many chunks on copy-engine streams, so a Map computes chunk k
 * while chunk k+1 uploads and its output streams back per chunk; 1..64,
 * default 8), "xfer_taper" (1 = the last two chunks are 1/2 and 1/4 of the
 * others, shortening the compute + download tail after the last upload;
 * default 1), "combine_peer" (copy(+) -> block with every device in
 * this process: 1 = each device folds its slice straight out of the peers'
 * replicas in one kernel, no staging copy; logical devices of one GPU share one
 * launch; 2 = one kernel per device even then; 0 = slices exchanged into
 * staging, then folded; default 1),
 * "mo_tma" (1 = a 2-D MapOverlap block stages its tile with one TMA copy,
 * where TMA can describe the tile: 16-byte aligned rows, staged row <= 256
 * units of up to 8 bytes, <= 256 rows; 0 = per-thread cp.async staging;
 * default 1), "mo_kt" (TMA kernel: tiles per block, stacked vertically, all
 * copies issued when the block starts; 1..4, or 0 = automatic: 2 for functions
 * needing >= 64 registers, else 1; default 0), "mo_full" (2-D MapOverlap: 1 =
 * threads whose rows and packed stores are all in range run an apply loop
 * without per-row guards, 0 = never, -1 = with 2+ tiles per block; default -1),
 * "mo_ws" (1 = 2-D MapOverlap tiles are staged by a TMA producer warp into a
 * ring of "mo_ws_stages" shared-memory buffers consumed by the other warps of
 * resident blocks, where TMA can describe the tile: 16-byte aligned rows, staged
 * row <= 256 units; otherwise the one-tile-per-block kernel runs),
 * and the tuning keys "scan_variant", "scan_chunks", "scan_minb", "mo_rh",
 * "mo_cw", "mo_minb", "mo_ws_minb", "ap_bk", "combine_unroll".  Environment defaults: SKL_BLOCK_THREADS,
 * SKL_DEBUG_BOUNDS; SKL_CACHE_DIR keeps compiled cubins on disk.              */
skl_status skl_set_option(skl_ctx* ctx, const char* key, long long value);
/* Counters: "launches" (kernels this library launched), "compiles" (NVRTC runs),
 * "cache_hits", "h2d_bytes", "d2h_bytes", "p2p_bytes" (device-to-device copy
 * bytes), "halo_push_bytes" (halo bytes stored by MapOverlap kernels directly
 * into neighbour devices' memory), "disk_cache_hits" (cubins loaded from
 * SKL_CACHE_DIR instead of compiled), "tma_launches" (MapOverlap launches of
 * the TMA / warp-specialised kernel), "nccl_groups" (NCCL send/recv groups of
 * redistributions issued), "nccl_comm" (1 when an NCCL communicator exists). */
skl_status skl_get_counter(skl_ctx* ctx, const char* key, long long* value);
const char* skl_last_error(void);

/* ------------------------------------------------------------------ containers
 * Vector<T> / Matrix<T>: "when a container is created on the CPU,
 * memory is allocated on the GPUs automatically; when a container ... is
 * deleted, the memory allocated on the GPUs is freed automatically".  A matrix
 * is row-major (index j*width+i) and is distributed by rows (A2).     */
skl_status skl_vector_create(skl_ctx* ctx, skl_type t, size_t n, skl_cont** out);
skl_status skl_matrix_create(skl_ctx* ctx, skl_type t, size_t rows, size_t cols, skl_cont** out);
skl_status skl_cont_destroy(skl_cont* c);
/* rows = n and cols = 1 for a vector.                                          */
skl_status skl_cont_info(skl_cont* c, skl_type* t, size_t* rows, size_t* cols, int* is_matrix);

/* Implicit transfers.  skl_copy_in writes the whole container
 * from `host` (bytes must equal the container size): if a distribution is set
 * the data goes straight to the devices that need it (no host mirror), else it
 * lands in the host mirror and is uploaded by the first skeleton that reads it.
 * skl_copy_out downloads the whole container into `host` (collective in
 * multi-process mode).  skl_copy_out_part downloads only the part that local
 * device g owns (its block rows/elements); first_unit / nunits say which.     */
skl_status skl_copy_in(skl_cont* c, const void* host, size_t bytes);
skl_status skl_copy_out(skl_cont* c, void* host, size_t bytes);
skl_status skl_copy_out_part(skl_cont* c, int g, void* host, size_t bytes, size_t* first_unit,
                             size_t* nunits);
/* Host view ("vec[i] = i"): a pinned mirror of the whole container.
 * SKL_READ downloads it if devices are newer; SKL_WRITE / SKL_RW mark the device
 * copies stale.  Valid until the next call that writes c, or its destruction.  */
#define SKL_READ 1
#define SKL_WRITE 2
#define SKL_RW 3
skl_status skl_host_data(skl_cont* c, int mode, void** host);
/* Fill every element with *value (on the devices of the current distribution;
 * a container with no distribution is filled in the host mirror).             */
skl_status skl_fill(skl_cont* c, const void* value);

/* ------------------------------------------------------------------ distributions
 * P:L205-222 (Figs. 1, 2): single (whole container on one GPU, the first by
 * default), copy (full replica on every GPU), block (contiguous disjoint chunk
 * per GPU; chunk = ceil(units/G), A1), overlap (block plus `arg` border units of
 * each neighbour; rows for a matrix).  P:L223-231: changing the distribution at
 * run time moves the data implicitly, device to device.
 *
 * `combine` (copy only; A25, BASELINE north_star): a Reduce skeleton whose
 * binary function (+) folds diverged replicas when the container leaves the copy
 * distribution: block g = r_0[g] (+) r_1[g] (+) ... (+) r_{G-1}[g], GPU order.
 * Replicas diverge when a skeleton writes the container as an extra argument
 * (SKL_WRITE) on several devices.  NULL = replicas are assumed identical.      */
#define SKL_DIST_NONE 0
#define SKL_SINGLE 1
#define SKL_COPY 2
#define SKL_BLOCK 3
#define SKL_OVERLAP 4
skl_status skl_set_distribution(skl_cont* c, int kind, int arg, skl_skel* combine);
skl_status skl_get_distribution(skl_cont* c, int* kind, int* arg);
/* Borrowed device view of device g's part: *dptr addresses unit *first_unit;
 * *nunits units are valid (including valid halo units for overlap).  For
 * tests and interop; NULL dptr if g holds nothing or is not local.            */
skl_status skl_local_part(skl_cont* c, int g, void** dptr, size_t* first_unit, size_t* nunits);

/* ------------------------------------------------------------------ skeletons
 * Customising functions are source strings (P:L252-254, P:L279-282,
 * P:L626-633), compiled at skeleton creation with NVRTC for sm_100a
 * (-fmad=false, IEEE div/sqrt, no FTZ: the GPU twin of the oracle's
 * -ffp-contract=off) and spliced into the skeleton's kernel.  The language is
 * CUDA C++ device code plus a compatibility prelude: uchar, uint, ushort,
 * `__global` (ignored), get(p,dx,dy) / get(p,dx) and SCL_NEUTRAL / SCL_NEAREST
 * (A14).  Functions need no __device__ qualifier.  `entry` names the function
 * to apply; NULL = the last top-level function defined in `src` (A13).
 *
 *  Map        P:L249-256   out[i] = f(in[i]);  out type SKL_VOID allowed (A27)
 *  Zip        P:L257-263   out[i] = l[i] (+) r[i]
 *  Reduce     P:L264-270   v1 (+) v2 (+) ... (+) vn, (+) associative only
 *  Scan       P:L271-278   inclusive prefix, (+) associative only (A9)
 *  MapOverlap P:L311-384   out[i,j] = f(&in[i,j]) with get(p,dx,dy), |dx|,|dy| <= d;
 *                          outside the matrix: `neutral` (SKL_NEUTRAL) or the
 *                          nearest valid element (SKL_NEAREST, A20)
 *
 * Extra arguments (A27, not in the paper): `extra[k]` types are appended to the
 * customising function's parameters; SKL_PTR-flagged ones are containers (the
 * function receives the local device's `T*`; a copy-distributed container is
 * the device's replica), others are passed by value.                          */
#define SKL_NEUTRAL 0
#define SKL_NEAREST 1
skl_status skl_map_create(skl_ctx* ctx, const char* src, const char* entry, skl_type in,
                          skl_type out, const skl_type* extra, int nextra, skl_skel** sk);
skl_status skl_zip_create(skl_ctx* ctx, const char* src, const char* entry, skl_type left,
                          skl_type right, skl_type out, const skl_type* extra, int nextra,
                          skl_skel** sk);
skl_status skl_reduce_create(skl_ctx* ctx, const char* src, const char* entry, skl_type t,
                             skl_skel** sk);
skl_status skl_scan_create(skl_ctx* ctx, const char* src, const char* entry, skl_type t,
                           skl_skel** sk);
skl_status skl_mapoverlap_create(skl_ctx* ctx, const char* src, const char* entry, skl_type in,
                                 skl_type out, int d, int boundary, const void* neutral,
                                 skl_skel** sk);
skl_status skl_skel_destroy(skl_skel* sk);
/* MapOverlap: *proven = 1 if every get() offset in the customising function was
 * proven within [-d, d] at creation (literal offsets, or counted for-loops with
 * literal bounds as in Listing 1.2) - the static check the paper names as future
 * work; 0 if not provable (a provable violation already made
 * skl_mapoverlap_create fail with SKL_ERR_OUT_OF_RANGE).                     */
skl_status skl_mapoverlap_bounds(skl_skel* sk, int* proven);

/* Allpairs: for an n x d matrix A and an
 * m x d matrix B, C (n x m) has C[i][j] = A_i (+) B_j over rows.
 * skl_allpairs_create: the customising function receives both rows and d,
 *   `TOUT f(const TIN* a, const TIN* b, int d)` (reading A35).
 * skl_allpairs_zr_create: C[i][j] = fold((+), zip((x), A_i, B_j)) with two
 *   binary customising functions - z = zip(a_k, b_k) (TIN x TIN -> TOUT) and
 *   the left fold acc = z_0, acc = (+)(acc, z_k) (TOUT x TOUT -> TOUT), e.g. the
 *   Manhattan distance or dotProduct (Eq. (1)); register-tiled on the
 *   FP32 pipes, each element folded in k order (reading A36).
 * Distributions: A as set (default block rows), B made copy, C like A.       */
skl_status skl_allpairs_create(skl_ctx* ctx, const char* src, const char* entry, skl_type in,
                               skl_type out, skl_skel** sk);
skl_status skl_allpairs_zr_create(skl_ctx* ctx, const char* zip_src, const char* zip_entry,
                                  const char* reduce_src, const char* reduce_entry, skl_type in,
                                  skl_type out, skl_skel** sk);
skl_status skl_allpairs_run(skl_skel* sk, skl_cont* A, skl_cont* B, skl_cont** C);

/* One extra argument at run time.                                             */
#define SKL_ARG_SCALAR 1
#define SKL_ARG_CONT 2
typedef struct skl_arg {
  int kind;          /* SKL_ARG_SCALAR or SKL_ARG_CONT                        */
  int mode;          /* containers: SKL_READ, SKL_WRITE or SKL_RW             */
  const void* value; /* scalars: pointer to the value (host)                  */
  size_t bytes;      /* scalars: size of the value                            */
  skl_cont* cont;    /* containers                                            */
} skl_arg;

/* Execution: `*out` NULL = allocate a new output container; otherwise it is
 * reused (must have the right type and size).  Distributions (A6-A8): inputs
 * without one default to block (MapOverlap: overlap(d)); Zip redistributes its
 * right input to the left one's; outputs take the input's distribution, except
 * MapOverlap (block) and Reduce (a 1-element scalar: single(0) with one process,
 * copy across processes).  A copy input is computed whole on every device.     */
skl_status skl_map_run(skl_skel* sk, skl_cont* in, skl_cont** out, const skl_arg* extra, int nextra);
skl_status skl_zip_run(skl_skel* sk, skl_cont* left, skl_cont* right, skl_cont** out,
                       const skl_arg* extra, int nextra);
skl_status skl_reduce_run(skl_skel* sk, skl_cont* in, skl_cont** scalar);
skl_status skl_scan_run(skl_skel* sk, skl_cont* in, skl_cont** out);
skl_status skl_mapoverlap_run(skl_skel* sk, skl_cont* in, skl_cont** out);
/* Scalar<T>::getValue(): download the 1-element result.           */
skl_status skl_scalar_get(skl_cont* scalar, void* value, size_t bytes);

/* ------------------------------------------------------------------ CUDA graphs
 * Record a sequence of skeleton calls once and replay it with one launch (for
 * latency-bound steps; the paper's runtime has no equivalent).  Between
 * skl_capture_begin and skl_capture_end the calls are recorded on the device
 * stream instead of executed; calls that hand data to the host (copy_out,
 * scalar_get, host_data, sync) are not allowed inside.  Containers and
 * skeletons used by a graph must outlive it, keep their sizes and
 * distributions, and have been used once before capture (so that nothing is
 * allocated or compiled while capturing).  Several local devices (one process
 * driving every GPU, or logical devices): the capture forks from the first
 * device's stream into the others and joins them at the end, so one launch
 * replays the whole multi-device sequence, halo exchanges included.  Not in
 * the one-process-per-GPU mode (skl_init_dist): SKL_ERR_UNSUPPORTED.         */
typedef struct skl_graph skl_graph;
skl_status skl_capture_begin(skl_ctx* ctx);
skl_status skl_capture_end(skl_ctx* ctx, skl_graph** out);
skl_status skl_graph_launch(skl_graph* g);
skl_status skl_graph_destroy(skl_graph* g);

/* ------------------------------------------------------------------ offline compilation
 * skl_init_offline: a context without devices (no GPU needed) in which
 * skeleton creation runs the full NVRTC compilation for sm_100a but loads
 * nothing; containers and skeleton calls fail with SKL_ERR_CUDA.  Used for
 * compile tests and for SASS inspection of the generated
 * kernels.  skl_skel_cubin copies the skeleton's sm_100a cubin (main program)
 * into buf (if cap suffices) and returns its size; skl_skel_source does the same
 * for the generated CUDA source.                                               */
skl_status skl_init_offline(skl_ctx** out);
skl_status skl_skel_cubin(skl_skel* sk, void* buf, size_t cap, size_t* size);
skl_status skl_skel_source(skl_skel* sk, char* buf, size_t cap, size_t* size);

/* ------------------------------------------------------------------ host-only planning
 * Pure host logic (no GPU needed), exported for tests of the multi-device path.
 * skl_plan_range: the unit range [lo,hi) device g must hold for a distribution
 * over `units` units and G devices (kind/arg as in skl_set_distribution;
 * `with_halo` = include overlap halos).
 * skl_plan_transfers: the device-to-device transfers that turn distribution
 * (from_kind, from_arg) into (to_kind, to_arg); written as 5-tuples
 * (src_device, src_unit, dst_device, dst_unit, nunits) in canonical order (the
 * order both sides of an NCCL send/recv pair issue them).  Returns the count in
 * *ntransfers (at most cap are written).                                       */
skl_status skl_plan_range(size_t units, int G, int kind, int arg, int g, int with_halo,
                          size_t* lo, size_t* hi);
skl_status skl_plan_transfers(size_t units, int G, int from_kind, int from_arg, int to_kind,
                              int to_arg, int64_t* tuples, size_t cap, size_t* ntransfers);

#ifdef __cplusplus
}
#endif
#endif /* SKL_H */

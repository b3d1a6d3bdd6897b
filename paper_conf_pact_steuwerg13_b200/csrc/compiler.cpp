// compiler.cpp — the customisation compiler (SURVEY §1 layer B4).
//
// P:L252-254 / P:L626-633: customising functions "are defined as plain strings"
// and compiled at run time (OpenCL's compiler in the paper).  Here: prelude +
// struct declarations + per-instantiation #defines + user source + skeleton
// kernel template -> NVRTC for sm_100a -> cubin -> cudaLibrary (context
// independent, valid on every device) -> cudaKernel_t.  Programs are cached by
// their full source text, so re-creating a skeleton costs nothing.
//
// Floating-point flags pin IEEE semantics (the GPU twin of the oracle's
// -ffp-contract=off): -fmad=false, --prec-div=true, --prec-sqrt=true, --ftz=false.
//
// NVRTC is loaded with dlopen on first use (libskl.so has no link-time CUDA
// driver or NVRTC dependency, so it loads on GPU-less hosts for ABI tests).
#include <dlfcn.h>

#include <cctype>
#include <mutex>

#include "skl_internal.h"

namespace skl {

extern const char* skl_embedded_kernels[];  // name, source, name, source, ..., nullptr

std::string kernel_template(const char* name) {
  for (int i = 0; skl_embedded_kernels[i]; i += 2)
    if (std::strcmp(skl_embedded_kernels[i], name) == 0) return skl_embedded_kernels[i + 1];
  fail(SKL_ERR_INVALID_ARG, std::string("missing kernel template ") + name);
}

namespace {
typedef int nvrtcResult_t;
struct Nvrtc {
  void* h = nullptr;
  nvrtcResult_t (*create)(void**, const char*, const char*, int, const char* const*, const char* const*);
  nvrtcResult_t (*compile)(void*, int, const char* const*);
  nvrtcResult_t (*logsize)(void*, size_t*);
  nvrtcResult_t (*log)(void*, char*);
  nvrtcResult_t (*cubinsize)(void*, size_t*);
  nvrtcResult_t (*cubin)(void*, char*);
  nvrtcResult_t (*destroy)(void**);
  const char* (*errstr)(nvrtcResult_t);
  nvrtcResult_t (*version)(int*, int*);
};
Nvrtc* nvrtc() {
  static Nvrtc n;
  static std::once_flag once;
  std::call_once(once, [] {
    const char* names[] = {"libnvrtc.so.12", "/usr/local/cuda/lib64/libnvrtc.so.12",
                           "/usr/local/cuda/lib64/libnvrtc.so", "libnvrtc.so"};
    for (const char* nm : names) {
      n.h = dlopen(nm, RTLD_NOW | RTLD_LOCAL);
      if (n.h) break;
    }
    if (!n.h) return;
    n.create = (decltype(n.create))dlsym(n.h, "nvrtcCreateProgram");
    n.compile = (decltype(n.compile))dlsym(n.h, "nvrtcCompileProgram");
    n.logsize = (decltype(n.logsize))dlsym(n.h, "nvrtcGetProgramLogSize");
    n.log = (decltype(n.log))dlsym(n.h, "nvrtcGetProgramLog");
    n.cubinsize = (decltype(n.cubinsize))dlsym(n.h, "nvrtcGetCUBINSize");
    n.cubin = (decltype(n.cubin))dlsym(n.h, "nvrtcGetCUBIN");
    n.destroy = (decltype(n.destroy))dlsym(n.h, "nvrtcDestroyProgram");
    n.errstr = (decltype(n.errstr))dlsym(n.h, "nvrtcGetErrorString");
    n.version = (decltype(n.version))dlsym(n.h, "nvrtcVersion");
  });
  if (!n.h || !n.create || !n.compile || !n.cubin)
    fail(SKL_ERR_UNSUPPORTED, "NVRTC (libnvrtc.so.12) could not be loaded");
  return &n;
}
}  // namespace

std::string program_source(Ctx* ctx, const std::string& body) {
  std::string s;
  s += "// ---- prelude (paper-compatibility, SURVEY §8(b))\n";
  s += kernel_template("prelude.cuh");
  s += "\n// ---- user types\n";
  for (const TypeInfo& t : ctx->types)
    if (!t.decl.empty()) s += t.decl + "\n";
  s += body;
  return s;
}

// ---- optional on-disk cubin cache (SKL_CACHE_DIR): a process that creates the
// same skeletons again skips NVRTC.  Key = two independent 64-bit hashes of the
// options, the NVRTC version and the full program source.
static const char* const kNvrtcOpts[] = {"--gpu-architecture=sm_100a", "-fmad=false", "--prec-div=true",
                                         "--prec-sqrt=true", "--ftz=false", "-default-device", "-std=c++17",
                                         "-lineinfo", "--extra-device-vectorization"};
static std::string cache_path(const std::string& source, int nvrtc_version) {
  const char* dir = std::getenv("SKL_CACHE_DIR");
  if (!dir || !*dir) return std::string();
  std::string text = std::to_string(nvrtc_version) + "\n";
  for (const char* o : kNvrtcOpts) text += std::string(o) + "\n";
  text += source;
  unsigned long long h1 = 1469598103934665603ull, h2 = 0x9e3779b97f4a7c15ull;
  for (unsigned char ch : text) {
    h1 = (h1 ^ ch) * 1099511628211ull;                          // FNV-1a
    h2 = (h2 ^ (ch + 0x9e3779b97f4a7c15ull + (h2 << 6) + (h2 >> 2))) * 0xff51afd7ed558ccdull;
  }
  char name[64];
  std::snprintf(name, sizeof(name), "/skl_%016llx%016llx.cubin", h1, h2);
  return std::string(dir) + name;
}
static bool cache_read(const std::string& path, std::vector<char>& out) {
  if (path.empty()) return false;
  FILE* f = std::fopen(path.c_str(), "rb");
  if (!f) return false;
  std::fseek(f, 0, SEEK_END);
  const long n = std::ftell(f);
  std::fseek(f, 0, SEEK_SET);
  bool ok = n > 0;
  if (ok) {
    out.resize((size_t)n);
    ok = std::fread(out.data(), 1, (size_t)n, f) == (size_t)n;
  }
  std::fclose(f);
  return ok;
}
static void cache_write(const std::string& path, const std::vector<char>& cubin) {
  if (path.empty()) return;
  const std::string tmp = path + ".tmp" + std::to_string((long long)getpid());
  FILE* f = std::fopen(tmp.c_str(), "wb");
  if (!f) return;  // the cache is an optimisation only
  const bool ok = std::fwrite(cubin.data(), 1, cubin.size(), f) == cubin.size();
  std::fclose(f);
  if (ok) std::rename(tmp.c_str(), path.c_str());  // atomic publish
  else std::remove(tmp.c_str());
}

Program* compile(Ctx* ctx, const std::string& source, std::string* log_out) {
  auto it = ctx->programs.find(source);
  if (it != ctx->programs.end()) {
    ctx->n_cache_hit++;
    return it->second.get();
  }
  Nvrtc* N = nvrtc();
  int vmaj = 0, vmin = 0;
  if (N->version) N->version(&vmaj, &vmin);
  const std::string cpath = cache_path(source, vmaj * 100 + vmin);
  {
    auto P = std::make_unique<Program>();
    if (cache_read(cpath, P->cubin)) {
      P->source = source;
      if (!ctx->offline) {
        ctx->set_device(ctx->first_local);
        SKL_CUDA(cudaLibraryLoadData(&P->lib, P->cubin.data(), nullptr, nullptr, 0, nullptr, nullptr, 0));
      }
      ctx->n_disk_hit++;
      Program* raw = P.get();
      ctx->programs[source] = std::move(P);
      return raw;
    }
  }
  void* prog = nullptr;
  if (N->create(&prog, source.c_str(), "skl_program.cu", 0, nullptr, nullptr) != 0)
    fail(SKL_ERR_COMPILE, "nvrtcCreateProgram failed");
  const int rc = N->compile(prog, (int)(sizeof(kNvrtcOpts) / sizeof(kNvrtcOpts[0])), kNvrtcOpts);
  size_t ls = 0;
  N->logsize(prog, &ls);
  std::string log(ls, '\0');
  if (ls) N->log(prog, &log[0]);
  if (log_out) *log_out = log;
  if (rc != 0) {
    N->destroy(&prog);
    fail(SKL_ERR_COMPILE, std::string("NVRTC: ") + (N->errstr ? N->errstr(rc) : "error") + "\n" + log);
  }
  auto P = std::make_unique<Program>();
  P->source = source;
  size_t cs = 0;
  N->cubinsize(prog, &cs);
  P->cubin.resize(cs);
  N->cubin(prog, P->cubin.data());
  N->destroy(&prog);
  if (!ctx->offline) {
    ctx->set_device(ctx->first_local);
    SKL_CUDA(cudaLibraryLoadData(&P->lib, P->cubin.data(), nullptr, nullptr, 0, nullptr, nullptr, 0));
  }
  ctx->n_compile++;
  cache_write(cpath, P->cubin);
  Program* raw = P.get();
  ctx->programs[source] = std::move(P);
  return raw;
}

// The dynamic shared-memory limit is a per-device attribute of the kernel: it is
// raised once per (physical device, kernel), so a second GPU gets it as well.
static cudaKernel_t get_kernel(Program* prog, int phys, const char* kernel, size_t smem) {
  auto it = prog->kernels.find(kernel);
  cudaKernel_t k;
  if (it == prog->kernels.end()) {
    SKL_CUDA(cudaLibraryGetKernel(&k, prog->lib, kernel));
    prog->kernels[kernel] = k;
  } else {
    k = it->second;
  }
  if (smem > 16 * 1024) {  // static + dynamic may exceed the 48 KB default: raise the limit
    const std::string key = std::to_string(phys) + "/" + kernel;
    auto s = prog->smem_set.find(key);
    if (s == prog->smem_set.end() || s->second < smem) {
      SKL_CUDA(cudaKernelSetAttributeForDevice(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem, phys));
      prog->smem_set[key] = smem;
    }
  }
  return k;
}

// Resident blocks per SM for a kernel at a block size / dynamic smem (persistent grids).
int occupancy(Ctx* ctx, int g, Program* prog, const char* kernel, int block, size_t smem) {
  const int phys = ctx->D(g).phys;
  const std::string key = std::to_string(phys) + "/" + kernel + "/" + std::to_string(block) + "/" +
                          std::to_string(smem);
  auto it = prog->occ.find(key);
  if (it != prog->occ.end()) return it->second;
  ctx->set_device(g);
  cudaKernel_t k = get_kernel(prog, phys, kernel, smem);
  int nb = 0;
  SKL_CUDA(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, (const void*)k, block, smem));
  prog->occ[key] = nb;
  return nb;
}

void launch(Ctx* ctx, int g, Program* prog, const char* kernel, dim3 grid, dim3 block, size_t smem,
            void** args) {
  if (grid.x == 0 || grid.y == 0 || grid.z == 0) return;
  Device& D = ctx->D(g);
  ctx->set_device(g);
  cudaKernel_t k = get_kernel(prog, D.phys, kernel, smem);
  SKL_CUDA(cudaLaunchKernel((const void*)k, grid, block, args, smem, D.stream));
  ctx->n_launch++;
}

// Reading A13: with no explicit entry, the customising function is the last
// top-level function *defined* in the source ("float func(...)",
// "float sum(...)", "float mult(...)": P:L254).
// the source without comments and string / char literals
static std::string strip_source(const std::string& src) {
  std::string s;
  s.reserve(src.size());
  for (size_t i = 0; i < src.size(); ++i) {
    if (src[i] == '/' && i + 1 < src.size() && src[i + 1] == '/') {
      while (i < src.size() && src[i] != '\n') ++i;
      s += '\n';
    } else if (src[i] == '/' && i + 1 < src.size() && src[i + 1] == '*') {
      i += 2;
      while (i + 1 < src.size() && !(src[i] == '*' && src[i + 1] == '/')) ++i;
      ++i;
      s += ' ';
    } else if (src[i] == '"' || src[i] == '\'') {
      const char q = src[i++];
      while (i < src.size() && src[i] != q) {
        if (src[i] == '\\') ++i;
        ++i;
      }
      s += ' ';
    } else {
      s += src[i];
    }
  }
  return s;
}

std::string detect_entry(const std::string& src) {
  const std::string s = strip_source(src);
  std::string last;
  int depth = 0;
  for (size_t i = 0; i < s.size(); ++i) {
    const char c = s[i];
    if (c == '{') {
      if (depth == 0) {
        // look back: ')' [qualifiers] '{'  -> find matching '(' and the identifier before it
        long j = (long)i - 1;
        while (j >= 0 && std::isspace((unsigned char)s[j])) --j;
        // skip trailing qualifiers such as const / noexcept
        while (j >= 0 && (std::isalnum((unsigned char)s[j]) || s[j] == '_')) {
          long k = j;
          while (k >= 0 && (std::isalnum((unsigned char)s[k]) || s[k] == '_')) --k;
          j = k;
          while (j >= 0 && std::isspace((unsigned char)s[j])) --j;
        }
        if (j >= 0 && s[j] == ')') {
          int pd = 0;
          for (; j >= 0; --j) {
            if (s[j] == ')') ++pd;
            else if (s[j] == '(' && --pd == 0) break;
          }
          --j;
          while (j >= 0 && std::isspace((unsigned char)s[j])) --j;
          long e = j;
          while (j >= 0 && (std::isalnum((unsigned char)s[j]) || s[j] == '_')) --j;
          if (e > j) {
            std::string name = s.substr((size_t)(j + 1), (size_t)(e - j));
            if (name != "if" && name != "for" && name != "while" && name != "switch") last = name;
          }
        }
      }
      ++depth;
    } else if (c == '}') {
      --depth;
    }
  }
  if (last.empty()) fail(SKL_ERR_COMPILE, "no function definition found in the customising source");
  return last;
}

}  // namespace skl

namespace skl {
void program_unload(Program* p) {
  if (p && p->lib) cudaLibraryUnload(p->lib);
  if (p) p->lib = nullptr;
}

// Debug bounds (A21): every program compiled with SKL_DEBUG_BOUNDS exports
// skl_bounds_flag; read and clear them after a MapOverlap launch.
bool read_and_clear_bounds_flags(Ctx* ctx) {
  bool hit = false;
  for (auto& d : ctx->dev) {
    SKL_CUDA(cudaSetDevice(d.phys));
    SKL_CUDA(cudaStreamSynchronize(d.stream));
  }
  for (auto& kv : ctx->programs) {
    Program* p = kv.second.get();
    void* dptr = nullptr;
    size_t sz = 0;
    if (cudaLibraryGetGlobal(&dptr, &sz, p->lib, "skl_bounds_flag") != cudaSuccess) {
      cudaGetLastError();
      continue;
    }
    for (auto& d : ctx->dev) {
      SKL_CUDA(cudaSetDevice(d.phys));
      if (cudaLibraryGetGlobal(&dptr, &sz, p->lib, "skl_bounds_flag") != cudaSuccess) {
        cudaGetLastError();
        continue;
      }
      unsigned v = 0;
      SKL_CUDA(cudaMemcpy(&v, dptr, sizeof(v), cudaMemcpyDeviceToHost));
      if (v) {
        hit = true;
        v = 0;
        SKL_CUDA(cudaMemcpy(dptr, &v, sizeof(v), cudaMemcpyHostToDevice));
      }
    }
  }
  return hit;
}
// A customising function whose source holds a loop (for / while / do): its
// per-element cost may vary (Mandelbrot's escape loop, a ray walk), so a Map /
// Zip over it defaults to the warp-interleaved kernel with one element per
// lane (option map_auto; the A22 loop: 1.13 -> 0.94 ms, sweep_r02_mandel_plain.log).
bool has_loop(const std::string& src) {
  const std::string s = strip_source(src);
  for (size_t i = 0; i < s.size();) {
    if (std::isalpha((unsigned char)s[i]) || s[i] == '_') {
      size_t j = i;
      while (j < s.size() && (std::isalnum((unsigned char)s[j]) || s[j] == '_')) ++j;
      const std::string w = s.substr(i, j - i);
      if (w == "for" || w == "while" || w == "do") return true;
      i = j;
    } else {
      ++i;
    }
  }
  return false;
}

}  // namespace skl

// jit.cu — run-time specialisation of the plan-signature kernels (NVRTC).
//
// Ocelot compiles its OpenCL kernels at run time for the device it runs on (PAPER.md
// L310-313 §3.1, L630-633 §4.2).  The ahead-of-time build instantiates the bulk kernels of
// spec_device.cuh for the signatures of the benchmark plans only (fused_spec.cu); every
// other plan used to fall back to the interpreted unified kernel (k_sga<DynShape>: ~440
// instructions per row, 0.13 of the copy bandwidth on Q1 + MIN/MAX).  Here a plan that fits
// the signature scheme — at most one range predicate, at most two integer key columns
// (packed <= 64 bits), up to six value expressions over at most four 8-byte value columns
// (all int64 or all fp64), SUM / MIN / MAX per value — gets its signature derived from the
// plan, the kernel compiled by NVRTC for sm_100a from the embedded device headers (the same
// source nvcc compiles ahead of time), loaded with cudaLibraryLoadData and cached per
// signature for the life of the process.  First use of a signature pays the compile
// (~1-2 s); later calls launch directly.  NVRTC is loaded at run time (dlopen); without it,
// or with OCL_NO_JIT set, plans keep the unified kernel.
#include <dlfcn.h>
#include <stdio.h>
#include <string.h>

#include <map>
#include <mutex>
#include <string>

#include <nvrtc.h>

#include "launch.cuh"
#include "spec_device.cuh"

#include "jit_src.inc"

namespace ocl {

namespace {

// ---- NVRTC entry points (dlopen)
struct NvrtcApi {
  bool tried = false, ok = false;
  decltype(&nvrtcCreateProgram) CreateProgram = nullptr;
  decltype(&nvrtcAddNameExpression) AddNameExpression = nullptr;
  decltype(&nvrtcCompileProgram) CompileProgram = nullptr;
  decltype(&nvrtcGetLoweredName) GetLoweredName = nullptr;
  decltype(&nvrtcGetCUBINSize) GetCUBINSize = nullptr;
  decltype(&nvrtcGetCUBIN) GetCUBIN = nullptr;
  decltype(&nvrtcGetProgramLogSize) GetProgramLogSize = nullptr;
  decltype(&nvrtcGetProgramLog) GetProgramLog = nullptr;
  decltype(&nvrtcDestroyProgram) DestroyProgram = nullptr;
};

std::mutex g_jit_mu;
NvrtcApi g_rtc;

bool rtc_load() {
  if (g_rtc.tried) return g_rtc.ok;
  g_rtc.tried = true;
  const char* names[] = {"libnvrtc.so.12", "libnvrtc.so", "/usr/local/cuda/lib64/libnvrtc.so.12"};
  void* h = nullptr;
  for (const char* n : names)
    if ((h = dlopen(n, RTLD_NOW | RTLD_GLOBAL))) break;
  if (!h) return false;
#define OCL_RTC(f, n) if (!(g_rtc.f = (decltype(g_rtc.f))dlsym(h, n))) return false;
  OCL_RTC(CreateProgram, "nvrtcCreateProgram");
  OCL_RTC(AddNameExpression, "nvrtcAddNameExpression");
  OCL_RTC(CompileProgram, "nvrtcCompileProgram");
  OCL_RTC(GetLoweredName, "nvrtcGetLoweredName");
  OCL_RTC(GetCUBINSize, "nvrtcGetCUBINSize");
  OCL_RTC(GetCUBIN, "nvrtcGetCUBIN");
  OCL_RTC(GetProgramLogSize, "nvrtcGetProgramLogSize");
  OCL_RTC(GetProgramLog, "nvrtcGetProgramLog");
  OCL_RTC(DestroyProgram, "nvrtcDestroyProgram");
#undef OCL_RTC
  g_rtc.ok = true;
  return true;
}

// ---- a signature at run time (mirrors Sig<...> of spec_device.cuh)
struct RtSig {
  int PW = 0;
  bool PF64 = false;
  int K0W = 0, K1W = 0, NC = 0;
  bool F64 = false;
  int NV = 0;
  uint32_t ops[kMaxVals] = {};
};

constexpr uint32_t rt_kind(uint32_t o) { return o & 3; }
constexpr uint32_t rt_flags(uint32_t o) { return (o >> 11) & 7; }

// Acc<S>::bytes(L, T) rounded to 128 (tier_bytes for L > 0)
size_t rt_priv_bytes(const RtSig& s, int L, int T) {
  int nnar = 0, nwide = 0, ndbl = 0, nmm = 0;
  for (int v = 0; v < s.NV; ++v) {
    const uint32_t f = rt_flags(s.ops[v]);
    if (f & VS_SUM) {
      if (s.F64) ++ndbl;
      else if (rt_kind(s.ops[v]) == VX_COL) ++nnar;
      else ++nwide;
    }
    nmm += ((f & VS_MIN) ? 1 : 0) + ((f & VS_MAX) ? 1 : 0);
  }
  const int nmm64 = s.F64 ? nmm : 0, nmm32 = s.F64 ? 0 : nmm;
  const size_t slot = ((size_t)T * (4 + 8 * (nnar + nwide + ndbl + nmm64) + 4 * (nwide + nmm32)) + 15) / 16 * 16;
  return ((size_t)(L + (s.F64 ? 0 : 1)) * slot + 127) / 128 * 128;
}

// TabL<S>::BYTES_PER_SLOT
size_t rt_tab_slot_bytes(const RtSig& s) {
  int nf = 1;
  for (int v = 0; v < s.NV; ++v) {
    const uint32_t f = rt_flags(s.ops[v]);
    nf += ((f & VS_SUM) ? 2 : 0) + ((f & VS_MIN) ? 1 : 0) + ((f & VS_MAX) ? 1 : 0);
  }
  return 8 + 4 * (size_t)nf;
}

size_t rt_stage_bytes(const RtSig& s, int R) { return (size_t)R * (s.PW + s.K0W + s.K1W + 8 * s.NC); }

bool rt_cta_ok(const RtSig& s) {
  if (s.F64) return false;
  for (int v = 0; v < s.NV; ++v)
    if (rt_kind(s.ops[v]) != VX_COL) return false;
  return true;
}

// Derive the signature of a plan and fill the SpecPlan (the run-time counterpart of
// spec_match in fused_spec.cu: same column order, same clamped predicate bounds).
bool rt_sig_of(const Plan& g, RtSig* sig, SpecPlan* sp) {
  RtSig s;
  if (g.npreds > 1 || g.nkeys > 2 || g.nvals < 1 || g.nvals > kMaxVals || !g.vec_ok) return false;
  if (g.npreds == 1) {
    s.PW = g.preds[0].col.width;
    s.PF64 = g.preds[0].is_f64 != 0;
  }
  if (g.nkeys >= 1) s.K0W = g.keys[0].col.width;
  if (g.nkeys == 2) s.K1W = g.keys[1].col.width;
  if (8 * (s.K0W + s.K1W) > 64) return false;
  const void* cols[4];
  int nc = 0;
  auto idx = [&](const DevCol& c) -> int {
    for (int i = 0; i < nc; ++i)
      if (cols[i] == c.ptr) return i;
    if (nc == 4 || c.width != 8) return -1;
    cols[nc] = c.ptr;
    return nc++;
  };
  s.F64 = g.vals[0].is_f64 != 0;
  s.NV = g.nvals;
  for (int v = 0; v < g.nvals; ++v) {
    const DevValue& d = g.vals[v];
    if ((d.is_f64 != 0) != s.F64) return false;
    const int a = idx(d.a), b = d.expr >= OCL_EXPR_MUL_1MINUS ? idx(d.b) : 0,
              c = d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? idx(d.c) : 0;
    if (a < 0 || b < 0 || c < 0) return false;
    const uint32_t flags = (d.off_sum >= 0 ? VS_SUM : 0) | (d.off_min >= 0 ? VS_MIN : 0) | (d.off_max >= 0 ? VS_MAX : 0);
    if (flags == 0) return false;
    s.ops[v] = vop((uint32_t)d.expr, (uint32_t)a, (uint32_t)b, (uint32_t)c, flags);
  }
  for (int i = 0; i < nc; ++i) {
    int dt = -1;
    for (int v = 0; v < g.nvals; ++v) {
      const DevValue& d = g.vals[v];
      if (d.a.ptr == cols[i]) dt = d.a.dtype;
      if (d.expr >= OCL_EXPR_MUL_1MINUS && d.b.ptr == cols[i]) dt = d.b.dtype;
      if (d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS && d.c.ptr == cols[i]) dt = d.c.dtype;
    }
    if (dt != (s.F64 ? OCL_F64 : OCL_I64)) return false;
  }
  s.NC = nc;
  memset(sp, 0, sizeof(*sp));
  sp->g = g;
  sp->pcol = s.PW > 0 ? g.preds[0].col.ptr : nullptr;
  if (s.PW > 0 && s.PW < 8 && !s.PF64) {
    int64_t lo = g.preds[0].lo, hi = g.preds[0].hi;
    if (lo > hi || lo > INT32_MAX || hi < INT32_MIN) { sp->plo = 1; sp->phi = 0; }
    else { sp->plo = (int32_t)(lo < INT32_MIN ? INT32_MIN : lo); sp->phi = (int32_t)(hi > INT32_MAX ? INT32_MAX : hi); }
  }
  sp->k0 = s.K0W > 0 ? g.keys[0].col.ptr : nullptr;
  sp->k1 = s.K1W > 0 ? g.keys[1].col.ptr : nullptr;
  for (int i = 0; i < 4; ++i) sp->col[i] = i < nc ? cols[i] : nullptr;
  *sig = s;
  return true;
}

// The run-time size formulas agree with the compile-time ones (checked on the Q1 signature).
constexpr RtSig kQ1Check = [] {
  RtSig s;
  s.PW = 4; s.K0W = 1; s.K1W = 1; s.NC = 4; s.NV = 5;
  s.ops[0] = vop(VX_COL, 0); s.ops[1] = vop(VX_COL, 1); s.ops[2] = vop(VX_M1, 1, 2);
  s.ops[3] = vop(VX_M1P, 1, 2, 3); s.ops[4] = vop(VX_COL, 2);
  return s;
}();
using Q1CheckSig = Sig<4, false, 1, 1, 4, false, vop(VX_COL, 0), vop(VX_COL, 1), vop(VX_M1, 1, 2),
                       vop(VX_M1P, 1, 2, 3), vop(VX_COL, 2)>;

std::string sig_expr(const RtSig& s, int L, int T, int R, int NS, const char* kernel = "k_sga_bulk") {
  char buf[512];
  int n = snprintf(buf, sizeof(buf), "ocl::%s<ocl::Sig<%d, %s, %d, %d, %d, %s", kernel, s.PW, s.PF64 ? "true" : "false",
                   s.K0W, s.K1W, s.NC, s.F64 ? "true" : "false");
  for (int v = 0; v < s.NV; ++v) n += snprintf(buf + n, sizeof(buf) - n, ", %uu", s.ops[v]);
  snprintf(buf + n, sizeof(buf) - n, ">, %d, %d, %d, %d>", L, T, R, NS);
  return buf;
}

struct JitKernel {
  cudaKernel_t k = nullptr;
  bool failed = false;
  int attr_smem[kMaxDevices] = {};
  int blocks[kMaxDevices][8] = {};
};
std::map<std::string, JitKernel>& jit_cache() {
  static std::map<std::string, JitKernel> m;
  return m;
}

// Compile (once) and load the kernel named by `expr`; nullptr if NVRTC is unavailable or
// the compile fails (the failure is cached: the plan keeps the unified kernel).
JitKernel* jit_get(const std::string& expr) {
  std::lock_guard<std::mutex> lk(g_jit_mu);
  JitKernel& jk = jit_cache()[expr];
  if (jk.k || jk.failed) return jk.failed ? nullptr : &jk;
  jk.failed = true;
  if (!rtc_load()) return nullptr;
  const std::string src = "#include \"spec_device.cuh\"\n";
  nvrtcProgram prog;
  if (g_rtc.CreateProgram(&prog, src.c_str(), "ocl_jit.cu", kJitNumHeaders, kJitHeaders, kJitHeaderNames) !=
      NVRTC_SUCCESS)
    return nullptr;
  g_rtc.AddNameExpression(prog, expr.c_str());
  const char* opts[] = {"--gpu-architecture=sm_100a", "-std=c++17", "-DOCL_JIT=1"};
  const nvrtcResult rc = g_rtc.CompileProgram(prog, 3, opts);
  if (rc != NVRTC_SUCCESS || getenv("OCL_DEBUG")) {
    size_t ls = 0;
    g_rtc.GetProgramLogSize(prog, &ls);
    std::string log(ls, '\0');
    g_rtc.GetProgramLog(prog, &log[0]);
    fprintf(stderr, "[ocl] NVRTC %s for %s%s%s\n", rc == NVRTC_SUCCESS ? "ok" : "FAILED", expr.c_str(),
            ls > 1 ? ":\n" : "", ls > 1 ? log.c_str() : "");
  }
  if (rc != NVRTC_SUCCESS) {
    g_rtc.DestroyProgram(&prog);
    return nullptr;
  }
  const char* lowered = nullptr;
  size_t cs = 0;
  if (g_rtc.GetLoweredName(prog, expr.c_str(), &lowered) != NVRTC_SUCCESS || g_rtc.GetCUBINSize(prog, &cs) != NVRTC_SUCCESS) {
    g_rtc.DestroyProgram(&prog);
    return nullptr;
  }
  std::string cubin(cs, '\0');
  g_rtc.GetCUBIN(prog, &cubin[0]);
  const std::string name = lowered;
  g_rtc.DestroyProgram(&prog);
  cudaLibrary_t lib;
  if (cudaLibraryLoadData(&lib, cubin.data(), nullptr, nullptr, 0, nullptr, nullptr, 0) != cudaSuccess ||
      cudaLibraryGetKernel(&jk.k, lib, name.c_str()) != cudaSuccess) {
    cudaGetLastError();
    jk.k = nullptr;
    return nullptr;
  }
  jk.failed = false;
  return &jk;
}

bool jit_launch(JitKernel* jk, const SpecPlan& sp, size_t smem, int T, int R, int sms, cudaStream_t s,
                cudaError_t* err, int slot_class) {
  int d = 0;
  if (cudaGetDevice(&d) != cudaSuccess || d < 0 || d >= kMaxDevices) return false;
  const void* fn = (const void*)jk->k;
  if ((int)smem > jk->attr_smem[d]) {
    if (cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem) != cudaSuccess) {
      cudaGetLastError();
      return false;
    }
    jk->attr_smem[d] = (int)smem;
  }
  int& nb = jk->blocks[d][slot_class];
  if (nb == 0) {
    int b = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, fn, T + 32, smem) != cudaSuccess || b < 1) {
      cudaGetLastError();
      b = -1;
    }
    nb = b;
  }
  if (nb < 1) return false;
  int64_t grid = (int64_t)sms * nb;
  const int64_t chunks = sp.g.n / R;
  if (chunks < grid) grid = chunks;
  if (grid < 1) return false;
  void* args[] = {(void*)&sp};
  count_launch();
  *err = cudaLaunchKernel(fn, dim3((unsigned)grid), dim3((unsigned)(T + 32)), args, smem, s);
  return true;
}

}  // namespace

static_assert(sizeof(Q1CheckSig) > 0, "");

// The run-time formulas equal the compile-time layout (evaluated once, on first use).
static bool jit_self_check() {
  return rt_priv_bytes(kQ1Check, 4, 128) == (Acc<Q1CheckSig>::bytes(4, 128) + 127) / 128 * 128 &&
         rt_stage_bytes(kQ1Check, 512) == (size_t)BulkStage<Q1CheckSig, 512>::BYTES &&
         rt_tab_slot_bytes(kQ1Check) == (size_t)TabL<Q1CheckSig>::BYTES_PER_SLOT;
}

// Run-time specialised bulk kernel for a plan no compiled-in signature took; false if the
// plan does not fit the signature scheme, JIT is off, or compiling / launching failed.
// *kind: 90 = private slots, 91 = CTA table.
bool launch_fused_jit(const Plan& g, int sms, cudaStream_t s, cudaError_t* err, int* kind) {
  if (getenv("OCL_NO_JIT")) return false;
  static const bool sane = jit_self_check();
  if (!sane) return false;
  RtSig sig;
  SpecPlan sp;
  if (!rt_sig_of(g, &sig, &sp)) return false;
  sp.sparse_pct = spec_sparse_pct(g.n);
  auto a16 = [](const void* q) { return ((uintptr_t)q & 15) == 0; };
  if ((sig.PW > 0 && !a16(sp.pcol)) || (sig.K0W > 0 && !a16(sp.k0)) || (sig.K1W > 0 && !a16(sp.k1))) return false;
  for (int i = 0; i < sig.NC; ++i)
    if (!a16(sp.col[i])) return false;
  const int64_t eg = g.expected > 0 ? g.expected : 1;
  int L, T, R, NS = 2;
  size_t tier;
  if (eg <= kPrivSlots) {
    bool mm = false;
    for (int v = 0; v < sig.NV; ++v) mm = mm || (rt_flags(sig.ops[v]) & (VS_MIN | VS_MAX));
    L = kPrivSlots;
    T = sig.F64 ? 256 : 128;                       // the compiled-in choices: fp64 <256, 512, 2>, int
    R = sig.F64 || !mm ? 512 : 256;                // <128, 512, 2>, int with MIN/MAX <128, 256, 3>
    NS = sig.F64 || !mm ? 2 : 3;
    tier = rt_priv_bytes(sig, L, T);
    *kind = 90;
  } else if (rt_cta_ok(sig) && eg <= 2048) {
    TabPolicy tp;
    if (!tab_policy(eg, rt_tab_slot_bytes(sig), rt_stage_bytes(sig, 64) / 64, &tp)) return false;
    L = 0;
    T = tp.T;
    R = tp.R;
    NS = tp.NS;
    sp.tab_hb = tp.hb;
    sp.tab_nrep = tp.nrep;
    sp.mm_check = tp.mm_check;
    tier = (((size_t)tp.nrep << tp.hb) * rt_tab_slot_bytes(sig) + 127) / 128 * 128;
    *kind = 91;
  } else {
    return false;
  }
  if (sp.g.n < R) return false;
  JitKernel* jk = jit_get(sig_expr(sig, L, T, R, NS));
  if (!jk) return false;
  sp.sparse_pct = spec_twin_pct(sp.sparse_pct, sig.PW > 0, L > 0);
  JitKernel* jks = nullptr;                      // the select-compact-gather twin (k_sga_sparse)
  if (sig.PW > 0 && sp.sparse_pct > 0 && !(jks = jit_get(sig_expr(sig, L, T, R, NS, "k_sga_sparse"))))
    sp.sparse_pct = 0;
  const size_t smem = tier + (size_t)NS * rt_stage_bytes(sig, R);
  int sc = 0;
  for (uint32_t c = sp.tab_nrep << sp.tab_hb; c > 128 && sc < 7; c >>= 1) ++sc;
  if (jks) {
    if (!jit_launch(jks, sp, smem, T, R, sms, s, err, sc)) return false;
    if (*err != cudaSuccess) return true;
  }
  return jit_launch(jk, sp, smem, T, R, sms, s, err, sc);
}

}  // namespace ocl

// tridiag_api.cu -- host side of libtridiag.so: argument validation, dispatch
// to the sm_100a kernels, launch configuration, and the host-buffer pipeline.
// The C ABI is declared (and documented) in include/tridiag.h.
#include <cuda_runtime.h>

#include <algorithm>
#include <atomic>
#include <cstdint>
#include <cstdlib>
#include <cstring>
#include <map>
#include <mutex>
#include <tuple>
#include <vector>

#include "host_common.h"
#include "tridiag_device.cuh"  // tdg::kPCR / kRD, ilog2c

namespace tdg_host {
thread_local int g_last_launches = 0;
thread_local const void* g_kernel_log[kMaxKernelLog];
thread_local int g_kernel_log_len = 0;
}  // namespace tdg_host

namespace {

using namespace tdg_host;
using tdg::ilog2c;

bool is_pow2(int64_t v) { return v >= 1 && (v & (v - 1)) == 0; }
// Systems are solved at the next power of two >= max(n, 2) (ragged n is padded
// in the kernels, see load_ragged); everything below works on n_pad.
int64_t pad_n(int64_t n) { int64_t p = 2; while (p < n) p <<= 1; return p; }
int ilog2_64(int64_t v) { int l = 0; while ((int64_t(1) << l) < v) ++l; return l; }
bool is_hybrid(int algo) { return algo == TRIDIAG_CR_PCR || algo == TRIDIAG_CR_RD; }
size_t elem_size(int dtype) { return dtype == TRIDIAG_F64 ? 8 : 4; }

// ---------------------------------------------------------------------------
// Capacity: the inner PCR/RD of an m-system larger than
// one equation per lane runs in shared memory (9m resp. 13m elements, at most
// 227 KB per CTA); everything else is register resident.
// ---------------------------------------------------------------------------
int64_t max_inner_m(int dtype) { return dtype == TRIDIAG_F64 ? 2048 : 4096; }
int64_t max_n_cr(int dtype) { return dtype == TRIDIAG_F64 ? 4096 : 8192; }

// Tuned intermediate size for the hybrids when switch_level == 0, from the
// switch-level sweeps (profiles/r01_tune_plan.md; Fig 17 is the paper's
// version of this sweep).  On B200 every m that keeps the inner
// solve in registers (m <= lanes per system) runs at the HBM roofline within
// noise, and every larger m is 2-10x slower; so CR+PCR takes the largest
// register-resident m (fewest CR levels) and CR+RD the smallest m within 2% of
// the best time (8), because RD's error grows with m on dominant input
// (R24).
int lanes_per_system(int dtype, int64_t n);
bool cta_plan(int dtype, int64_t n);
int auto_m(int64_t n, int dtype, int algo) {
  if (!is_hybrid(algo)) return 0;
  const int64_t P = lanes_per_system(dtype, n);
  // CTA plans (n > 32 R): m = 32 for both hybrids.  For CR+RD, m = n / R (one
  // survivor per lane for the CTA-wide blocked scan) is 8-25% faster
  // (profiles/r01_rd_tune2.txt) but RD's error grows with m (R24: POI fp32
  // 2e-5 at m = 32, ~1e-3 at m = 256), so the table keeps the accurate m and
  // the fast one is the caller's choice.
  int64_t m = (algo == TRIDIAG_CR_PCR || cta_plan(dtype, n)) ? std::min<int64_t>(P, 32)
                                                             : std::min<int64_t>(P, 8);
  if (m < 2) m = 2;
  if (m > n) m = n;
  return (int)m;
}


// Tuning knobs (environment).  Read ONCE, on the first call of the library
// (std::call_once), into atomics: the launch plan never changes mid-process
// and no solve pays a getenv.  tridiag_reload_knobs() re-reads them (A/B
// measurements and the bitwise path-equality tests only).  Defaults are the
// tuned paths (profiles/r01_tune_plan.md):
//   TRIDIAG_WARP_R       force R of the warp kernel (0 = plan)
//   TRIDIAG_PREFETCH     L2 bulk prefetch of the next system (2 = auto)
//   TRIDIAG_CTA_DBUF     double-buffered CTA-kernel regions (1)
//   TRIDIAG_RAG_TMA      vector paths for ragged / pitched rows (1)
//   TRIDIAG_TMA_PF       TMA-box L2 prefetch of the unit after next (0)
//   TRIDIAG_SMALL_CTA    smaller warp-kernel CTAs for small batches (1)
//   TRIDIAG_PDL          programmatic dependent launch (1)
//   TRIDIAG_TMA          TMA CTA kernels (1)
//   TRIDIAG_BLOCKED_MINB blocked-inner register cap (2)
//   TRIDIAG_COL_TMA      TMA-fed column passes (1)
//   TRIDIAG_PHASE_STAMPS per-phase clock stamps (0)
//   TRIDIAG_PREWAIT_PF   L2 prefetch of the first system before the PDL wait (1)
//   TRIDIAG_COL_ORDER    chunk-major unit order of the column expansion pass (1)
int env_int(const char* name, int dflt) {
  const char* v = getenv(name);
  return (v && *v) ? atoi(v) : dflt;
}

enum Knob { kWarpR, kPrefetch, kCtaDbuf, kRagTma, kTmaPf, kSmallCta, kPdl, kTma, kBlockedMinb,
            kColTma, kPhaseStamps, kPrewaitPf, kColOrder, kNumKnobs };
struct KnobDef { const char* name; int dflt; };
constexpr KnobDef kKnobDefs[kNumKnobs] = {
    {"TRIDIAG_WARP_R", 0},    {"TRIDIAG_PREFETCH", 2},  {"TRIDIAG_CTA_DBUF", 1},
    {"TRIDIAG_RAG_TMA", 1},   {"TRIDIAG_TMA_PF", 0},    {"TRIDIAG_SMALL_CTA", 1},
    {"TRIDIAG_PDL", 1},       {"TRIDIAG_TMA", 1},       {"TRIDIAG_BLOCKED_MINB", 2},
    {"TRIDIAG_COL_TMA", 1},   {"TRIDIAG_PHASE_STAMPS", 0}, {"TRIDIAG_PREWAIT_PF", 1}, {"TRIDIAG_COL_ORDER", 1}};
std::atomic<int> g_knobs[kNumKnobs];
std::once_flag g_knobs_once;
std::mutex g_knobs_mu;

void read_knobs() {
  std::lock_guard<std::mutex> lk(g_knobs_mu);
  for (int i = 0; i < kNumKnobs; ++i)
    g_knobs[i].store(env_int(kKnobDefs[i].name, kKnobDefs[i].dflt), std::memory_order_relaxed);
}
int knob(Knob k) {
  std::call_once(g_knobs_once, read_knobs);
  return g_knobs[k].load(std::memory_order_relaxed);
}
int force_R() { return knob(kWarpR); }

}  // namespace

namespace tdg_host {

int prefetch_mode() { return knob(kPrefetch); }
int cta_dbuf_mode() { return knob(kCtaDbuf); }
int rag_tma_mode() { return knob(kRagTma); }
int tma_pf_mode() { return knob(kTmaPf); }
int small_cta_mode() { return knob(kSmallCta); }
int pdl_mode() { return knob(kPdl); }
int tma_mode() { return knob(kTma); }
int blocked_minb() { return knob(kBlockedMinb); }
int col_tma_mode() { return knob(kColTma); }
int prewait_pf_mode() { return knob(kPrewaitPf); }
int col_order_mode() { return knob(kColOrder); }

// Phase stamps (diagnostic, NEXT f4): one device buffer per launch slot of a
// call (slot = the launch's index within the call, as in the kernel log),
// grown on demand; tridiag_phase_stamps() copies the last launch's stamps
// back, tridiag_phase_stamps_of(i) those of launch i of the last call.
namespace {
std::mutex g_stamp_mu;
long long* g_stamp_dev[kMaxKernelLog] = {};
int64_t g_stamp_cap[kMaxKernelLog] = {}, g_stamp_len[kMaxKernelLog] = {};
}  // namespace
long long* stamp_buffer(int64_t elems) {
  if (!knob(kPhaseStamps)) return nullptr;
  const int slot = g_kernel_log_len;  // index of the launch about to be made
  if (slot >= kMaxKernelLog) return nullptr;
  std::lock_guard<std::mutex> lk(g_stamp_mu);
  if (elems > g_stamp_cap[slot]) {
    if (g_stamp_dev[slot]) cudaFree(g_stamp_dev[slot]);
    g_stamp_dev[slot] = nullptr;
    g_stamp_cap[slot] = 0;
    if (cudaMalloc(&g_stamp_dev[slot], elems * sizeof(long long)) != cudaSuccess) return nullptr;
    g_stamp_cap[slot] = elems;
  }
  cudaMemset(g_stamp_dev[slot], 0, elems * sizeof(long long));
  g_stamp_len[slot] = elems;
  return g_stamp_dev[slot];
}

// R per lane from the plan sweep (profiles/r01_tune_plan.md): on HBM-scale
// batches the widest register block that fits (16 fp32 / 8 fp64 equations per
// lane) is fastest at every n, and systems with n <= 32 use 4 lanes.  Small
// batches (fewer than ~8 warps' worth of lanes per SM at that R) are latency
// bound instead: they spread each system over more lanes (R = n/32, a full
// warp), which keeps m <= 32 on the register path.  num_systems < 0 asks for
// the HBM-scale plan.
constexpr int64_t kSmallBatchLanes = 148LL * 8 * 32;

Plan plan_for(int dtype, int64_t n, int64_t S) {
  const int fr = force_R();
  const int Rmax = dtype == TRIDIAG_F32 ? 16 : 8;
  if (fr > 0 && fr <= Rmax && fr <= n && n / fr <= 32 && (fr & (fr - 1)) == 0) return {false, fr, 0};
  if (n > 32 * Rmax) return {true, Rmax, (int)(n / (Rmax * 32))};
  int R = n <= 32 ? (int)std::max<int64_t>(1, n / 4) : Rmax;
  if (S >= 0 && S * n / R < kSmallBatchLanes) R = (int)std::max<int64_t>(1, n / 32);
  return {false, R, 0};
}

}  // namespace tdg_host

namespace {

// Lanes per system of the HBM-scale plan: the largest m the hybrids keep on
// the register path (the small-batch plan has at least as many lanes).
bool cta_plan(int dtype, int64_t n) { return plan_for(dtype, n).cta; }

int lanes_per_system(int dtype, int64_t n) {
  const Plan p = plan_for(dtype, n);
  return p.cta ? 32 : (int)(n / p.R);
}

struct Dev {
  int sms = 0;
};
std::mutex g_mu;
std::map<int, Dev> g_dev;

}  // namespace

namespace tdg_host {

std::mutex& occ_mutex() {
  static std::mutex m;
  return m;
}
std::map<std::tuple<int, const void*, int, size_t>, int>& occ_cache() {
  static std::map<std::tuple<int, const void*, int, size_t>, int> c;
  return c;
}

int device_sms(int dev) {
  std::lock_guard<std::mutex> lk(g_mu);
  Dev& D = g_dev[dev];
  if (D.sms == 0) cudaDeviceGetAttribute(&D.sms, cudaDevAttrMultiProcessorCount, dev);
  return D.sms;
}

// TMA tensor maps: driver entry point fetched once through the runtime.
PFN_cuTensorMapEncodeTiled_v12000 encode_fn() {
  static PFN_cuTensorMapEncodeTiled_v12000 fn = nullptr;
  static std::once_flag once;
  std::call_once(once, [] {
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      fn = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(p);
  });
  return fn;
}

}  // namespace tdg_host

namespace {

bool overlaps(const void* p, const void* q, size_t bytes) {
  const uintptr_t a = reinterpret_cast<uintptr_t>(p), b = reinterpret_cast<uintptr_t>(q);
  return a < b + bytes && b < a + bytes;
}

// Host-side argument validation (integer only; nothing is enqueued on error).
// On success *m_out is the resolved intermediate size m (n for PCR/RD, 2 for CR).
int validate(const void* a, const void* b, const void* c, const void* d, const void* x,
             int64_t n, int64_t S, int dtype, int algo, int switch_level, int64_t* m_out,
             int64_t es, int64_t ss, bool large = false) {
  // NULL pointers are legal only for an empty batch (nothing is accessed).
  if (S != 0 && (!a || !b || !c || !d || !x)) return TRIDIAG_ERR_NULL;
  if (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64) return TRIDIAG_ERR_DTYPE;
  if (algo < TRIDIAG_CR || algo > TRIDIAG_RD_STONE) return TRIDIAG_ERR_ALGO;
  if (n < 1) return TRIDIAG_ERR_N;
  const int64_t np = pad_n(n);
  if (np > (large ? tridiag_max_n_large(dtype, algo) : tridiag_max_n(dtype, algo)))
    return TRIDIAG_ERR_N_TOO_LARGE;
  if (S < 0) return TRIDIAG_ERR_NUM_SYSTEMS;
  int64_t m;
  if (algo == TRIDIAG_CR) m = 2;
  else if (algo == TRIDIAG_PCR || algo == TRIDIAG_RD || algo == TRIDIAG_RD_STONE) m = np;
  else m = switch_level == 0 ? tridiag_auto_switch_level(np, dtype, algo) : switch_level;
  if (!is_hybrid(algo) && switch_level != 0) return TRIDIAG_ERR_SWITCH_LEVEL;
  if (is_hybrid(algo) && large) {
    // resolved against the level plan by solve_large
    if (switch_level < 0 || (switch_level != 0 && (switch_level < 2 || !is_pow2(switch_level) ||
                                                   switch_level > np ||
                                                   switch_level > max_inner_m(dtype))))
      return TRIDIAG_ERR_SWITCH_LEVEL;
    m = switch_level;
  } else if (is_hybrid(algo)) {
    if (switch_level < 0 || m < 2 || !is_pow2(m) || m > np ||
        m > tridiag_max_switch_level(dtype, algo, np))
      return TRIDIAG_ERR_SWITCH_LEVEL;
  }
  // strides: element (s, i) at s*ss + i*es must be one-to-one (one index nests the other)
  if (es < 1 || ss < 1) return TRIDIAG_ERR_STRIDE;
  if (S > 1 && n > 1 && !(ss >= es * n || es >= ss * S)) return TRIDIAG_ERR_STRIDE;
  if (n > 1 && S > 1 && es > 1 && ss > 1) return TRIDIAG_ERR_STRIDE;  // one stride must be 1
  const size_t bytes = S > 0 ? (size_t)((S - 1) * ss + (n - 1) * es + 1) * elem_size(dtype) : 0;
  if (bytes > 0) {
    if (overlaps(x, a, bytes) || overlaps(x, b, bytes) || overlaps(x, c, bytes)) return TRIDIAG_ERR_OVERLAP;
    if (x != d && overlaps(x, d, bytes)) return TRIDIAG_ERR_OVERLAP;
  }
  *m_out = m;
  return TRIDIAG_OK;
}

// A single system (S <= 1) has no system stride, and a 1-equation system no
// element stride: map both onto the layout the kernels expect (contiguous
// when es == 1, else the interleaved layout with system stride 1), so the
// element stride is always honoured.  Multi-system layouts pass unchanged.
Layout normalise_layout(int64_t n, int64_t S, int64_t es, int64_t ss) {
  if (n <= 1) es = 1;
  if (S <= 1) ss = es == 1 ? n : 1;
  return Layout{es, ss};
}

int solve_device(const void* a, const void* b, const void* c, const void* d, void* x, int64_t nr,
                 int64_t S, int dtype, int algo, int64_t m, cudaStream_t st, Layout L) {
  if (S == 0) return TRIDIAG_OK;
  const int64_t n = pad_n(nr);
  const int k = ilog2_64(n / m);
  const int inner = (algo == TRIDIAG_RD || algo == TRIDIAG_CR_RD) ? tdg::kRD
                    : algo == TRIDIAG_RD_STONE                     ? tdg::kSTONE
                                                                   : tdg::kPCR;
  cudaError_t e;
  if (dtype == TRIDIAG_F32)
    e = inner == tdg::kPCR ? dispatch_t<float, tdg::kPCR>(a, b, c, d, x, n, S, k, st, dtype, nr, L)
        : inner == tdg::kRD ? dispatch_t<float, tdg::kRD>(a, b, c, d, x, n, S, k, st, dtype, nr, L)
                            : dispatch_t<float, tdg::kSTONE>(a, b, c, d, x, n, S, k, st, dtype, nr, L);
  else
    e = inner == tdg::kPCR ? dispatch_t<double, tdg::kPCR>(a, b, c, d, x, n, S, k, st, dtype, nr, L)
        : inner == tdg::kRD ? dispatch_t<double, tdg::kRD>(a, b, c, d, x, n, S, k, st, dtype, nr, L)
                            : dispatch_t<double, tdg::kSTONE>(a, b, c, d, x, n, S, k, st, dtype, nr, L);
  return e == cudaSuccess ? TRIDIAG_OK : (int)e;
}

// ---------------------------------------------------------------------------
// Large n (NEXT f2): reduction passes of log2 R CR levels each
// until the system fits the on-chip kernels (n <= bottom_n), the on-chip
// solve of the reduced system, then the expansion passes in reverse.
// ---------------------------------------------------------------------------
struct LargeLevel {
  int64_t n;  // padded size of this level's system
  int kin;    // CR levels applied by its pass
};
int large_R(int dtype) { return dtype == TRIDIAG_F64 ? 8 : 16; }
int64_t large_chunk_n(int dtype) {
  return dtype == TRIDIAG_F64 ? large_chunk<double>() : large_chunk<float>();
}
size_t align256(size_t v) { return (v + 255) & ~size_t(255); }

// Level plan for a padded size np and intermediate size m (2 for CR); false
// if bottom_n is not a valid stopping size for this dtype.
bool large_plan(int64_t np, int dtype, int64_t m, int64_t bottom_n, std::vector<LargeLevel>* lv,
                int64_t* n_last) {
  const int LR = ilog2_64(large_R(dtype));
  const int64_t CH = large_chunk_n(dtype);
  lv->clear();
  int64_t cur = np;
  while (cur > bottom_n) {
    const int kin = std::min(LR, ilog2_64(cur / m));
    if (kin < 1 || cur % CH != 0) return false;
    lv->push_back({cur, kin});
    cur >>= kin;
  }
  *n_last = cur;
  return true;
}

int64_t resolve_bottom_n(int dtype, int64_t bottom_n) {
  if (bottom_n == 0) return max_n_cr(dtype);
  if (!is_pow2(bottom_n) || bottom_n < large_chunk_n(dtype) / 2 || bottom_n > max_n_cr(dtype)) return -1;
  return bottom_n;
}

// m of a large solve: CR 2, PCR / RD n; hybrids the caller's m or the auto
// table at the size the passes reduce to.  -1 if invalid.
int64_t large_m(int64_t np, int dtype, int algo, int64_t m_req, int64_t bottom_n) {
  if (algo == TRIDIAG_CR) return 2;
  if (!is_hybrid(algo)) return np <= bottom_n ? np : -1;
  std::vector<LargeLevel> lv;
  int64_t n_last = 0;
  if (m_req == 0) {
    if (!large_plan(np, dtype, 2, bottom_n, &lv, &n_last)) return -1;
    m_req = auto_m(n_last, dtype, algo);
  }
  if (!large_plan(np, dtype, m_req, bottom_n, &lv, &n_last)) return -1;
  if (m_req > tridiag_max_switch_level(dtype, algo, n_last)) return -1;
  return m_req;
}

size_t large_ws_bytes(const std::vector<LargeLevel>& lv, int64_t S, int dtype) {
  const size_t T = elem_size(dtype);
  size_t total = 0;
  for (const LargeLevel& L : lv) {
    total += 4 * align256((size_t)S * (size_t)(L.n >> L.kin) * T);
  }
  return total;
}

template <typename T>
int solve_large_t(const T* a, const T* b, const T* c, const T* d, T* x, int64_t nr, int64_t S,
                  int dtype, int algo, int64_t m, const std::vector<LargeLevel>& lv,
                  int64_t n_last, char* ws, cudaStream_t st, int64_t ss0) {
  const T c_pad = (algo == TRIDIAG_CR_RD) ? T(1) : T(0);
  struct Buf { T* a; T* b; T* c; T* d; };
  std::vector<Buf> bufs;
  char* p = ws;
  for (const LargeLevel& L : lv) {
    const size_t arr = align256((size_t)S * (size_t)(L.n >> L.kin) * sizeof(T));
    Buf B;
    B.a = reinterpret_cast<T*>(p); B.b = reinterpret_cast<T*>(p + arr);
    B.c = reinterpret_cast<T*>(p + 2 * arr); B.d = reinterpret_cast<T*>(p + 3 * arr);
    p += 4 * arr;
    bufs.push_back(B);
  }
  auto al = [](const void* q) { return (reinterpret_cast<uintptr_t>(q) % 32) == 0; };
  int launches = 0;
  // forward: level j's inputs are the user's arrays (j = 0) or bufs[j - 1]
  for (size_t j = 0; j < lv.size(); ++j) {
    const LargeLevel& L = lv[j];
    const bool first = j == 0;
    const T* ia = first ? a : bufs[j - 1].a;
    const T* ib = first ? b : bufs[j - 1].b;
    const T* ic = first ? c : bufs[j - 1].c;
    const T* id = first ? d : bufs[j - 1].d;
    const int64_t n_real = first ? nr : L.n;
    const int64_t ss = first ? ss0 : L.n;
    const bool vec = n_real == L.n && al(ia) && al(ib) && al(ic) && al(id) &&
                     ((uint64_t)ss * sizeof(T)) % 32 == 0;
    const Buf& B = bufs[j];
    const cudaError_t e = large_pass<T>(1, ia, ib, ic, id, B.a, B.b, B.c, B.d, nullptr, L.n,
                                        n_real, ss, S, L.kin, vec, c_pad, st);
    if (e != cudaSuccess) return (int)e;
    launches += 1;
  }
  // on-chip solve of the reduced system, in place (x == d)
  const Buf& Z = bufs.back();
  const int rc = solve_device(Z.a, Z.b, Z.c, Z.d, Z.d, n_last, S, dtype, algo, m, st, Layout{1, n_last});
  if (rc != TRIDIAG_OK) return rc;
  launches += g_last_launches;
  // backward: level j writes x into the user's x (j = 0) or bufs[j - 1].d
  for (size_t jj = lv.size(); jj-- > 0;) {
    const LargeLevel& L = lv[jj];
    const bool first = jj == 0;
    const T* ia = first ? a : bufs[jj - 1].a;
    const T* ib = first ? b : bufs[jj - 1].b;
    const T* ic = first ? c : bufs[jj - 1].c;
    const T* id = first ? d : bufs[jj - 1].d;
    T* ox = first ? x : bufs[jj - 1].d;
    const int64_t n_real = first ? nr : L.n;
    const int64_t ss = first ? ss0 : L.n;
    const bool vec = n_real == L.n && al(ia) && al(ib) && al(ic) && al(id) && al(ox) &&
                     ((uint64_t)ss * sizeof(T)) % 32 == 0;
    const cudaError_t e = large_pass<T>(2, ia, ib, ic, id, ox, nullptr, nullptr, nullptr,
                                        bufs[jj].d, L.n, n_real, ss, S, L.kin, vec, c_pad, st);
    if (e != cudaSuccess) return (int)e;
    launches += 1;
  }
  g_last_launches = launches;
  return TRIDIAG_OK;
}

// ---------------------------------------------------------------------------
// Interleaved layouts with n > 32 R (the ADI column sweep, NEXT f1 + f2):
// column reduction passes (tridiag_colpass.cuh) -- at least one, then more
// until the system has at most `bottom` equations (default tridiag_max_n) --
// the last of which writes the survivors transposed into contiguous rows in
// the workspace; the row kernels solve those reduced systems; expansion
// passes back-substitute.
// ---------------------------------------------------------------------------
int64_t col_chunk_n(int dtype) { return dtype == TRIDIAG_F64 ? col_chunk<double>() : col_chunk<float>(); }
int64_t col_onchip_max(int dtype) { return 32 * large_R(dtype); }  // interleaved kernel capacity

int64_t resolve_col_bottom(int dtype, int64_t bottom_n) {
  if (bottom_n == 0) return max_n_cr(dtype);
  if (!is_pow2(bottom_n) || bottom_n < col_chunk_n(dtype) / 2 || bottom_n > max_n_cr(dtype)) return -1;
  return bottom_n;
}

bool col_plan(int64_t np, int dtype, int64_t m, int64_t bottom, std::vector<LargeLevel>* lv,
              int64_t* n_last) {
  const int LR = ilog2_64(large_R(dtype));
  const int64_t CH = col_chunk_n(dtype);
  lv->clear();
  int64_t cur = np;
  while (cur > bottom || lv->empty()) {
    const int kin = std::min(LR, ilog2_64(cur / m));
    if (kin < 1 || cur % CH != 0) return false;
    lv->push_back({cur, kin});
    cur >>= kin;
  }
  *n_last = cur;
  return !lv->empty();
}

// m of a column-pass solve (CR 2; hybrids the caller's m, else the tuned m of
// the full size -- the same default as the contiguous solve -- or, beyond the
// on-chip sizes, of the reduced size); -1 when no pass plan exists.
int64_t col_m(int64_t np, int dtype, int algo, int64_t m_req, int64_t bottom,
              std::vector<LargeLevel>* lv, int64_t* n_last) {
  if (algo == TRIDIAG_CR) {
    if (!col_plan(np, dtype, 2, bottom, lv, n_last)) return -1;
    return 2;
  }
  if (!is_hybrid(algo)) return -1;
  if (m_req == 0) {
    if (np <= max_n_cr(dtype)) {
      m_req = auto_m(np, dtype, algo);
    } else {
      if (!col_plan(np, dtype, 2, bottom, lv, n_last)) return -1;
      m_req = auto_m(*n_last, dtype, algo);
    }
  }
  if (!col_plan(np, dtype, m_req, bottom, lv, n_last)) return -1;
  if (m_req > tridiag_max_switch_level(dtype, algo, *n_last)) return -1;
  return m_req;
}

size_t col_ws_bytes(const std::vector<LargeLevel>& lv, int64_t S, int dtype) {
  const size_t T = elem_size(dtype);
  size_t total = 0;
  for (const LargeLevel& L : lv) total += 4 * align256((size_t)S * (size_t)(L.n >> L.kin) * T);
  return total;
}

// Pass plan of tridiag_solve_batched_strided_large.  kind: 0 = no passes
// (the on-chip strided path, m in *m), 1 = row passes (large-n plan),
// 2 = column passes; negative = status code.
struct StridedPlan {
  int kind = 0;
  int64_t m = 0, n_last = 0;
  std::vector<LargeLevel> lv;
};

// Workspace of a column plan: the passes' reduced levels.
size_t col_need(const StridedPlan& P, int64_t n, int64_t S, int dtype, int algo, int64_t bottom_n) {
  (void)n; (void)algo; (void)bottom_n;
  return col_ws_bytes(P.lv, S, dtype);
}

template <typename T>
int solve_col_t(const T* a, const T* b, const T* c, const T* d, T* x, int64_t nr, int64_t S,
                int64_t es, int dtype, int algo, int64_t m, const std::vector<LargeLevel>& lv,
                int64_t n_last, char* ws, cudaStream_t st) {
  const T c_pad = (algo == TRIDIAG_CR_RD) ? T(1) : T(0);
  struct Buf { T* a; T* b; T* c; T* d; };
  std::vector<Buf> bufs;
  char* p = ws;
  for (const LargeLevel& L : lv) {
    const size_t arr = align256((size_t)S * (size_t)(L.n >> L.kin) * sizeof(T));
    Buf B;
    B.a = reinterpret_cast<T*>(p); B.b = reinterpret_cast<T*>(p + arr);
    B.c = reinterpret_cast<T*>(p + 2 * arr); B.d = reinterpret_cast<T*>(p + 3 * arr);
    p += 4 * arr;
    bufs.push_back(B);
  }
  int launches = 0;
  for (size_t j = 0; j < lv.size(); ++j) {
    const LargeLevel& L = lv[j];
    const bool first = j == 0;
    const T* ia = first ? a : bufs[j - 1].a;
    const T* ib = first ? b : bufs[j - 1].b;
    const T* ic = first ? c : bufs[j - 1].c;
    const T* id = first ? d : bufs[j - 1].d;
    const Buf& B = bufs[j];
    // the last pass transposes its survivors into contiguous rows
    const bool last = j + 1 == lv.size();
    const cudaError_t e = col_pass<T>(1, ia, ib, ic, id, B.a, B.b, B.c, B.d, nullptr, L.n,
                                      first ? nr : L.n, first ? es : S, S, last ? 1 : S,
                                      last ? n_last : 1, L.kin, c_pad, st);
    if (e != cudaSuccess) return (int)e;
    launches += 1;
  }
  // the reduced systems, contiguous rows of n_last <= tridiag_max_n equations:
  // the row kernels (warp / TMA CTA), in place
  const Buf& Z = bufs.back();
  const int rc = solve_device(Z.a, Z.b, Z.c, Z.d, Z.d, n_last, S, dtype, algo, m, st, Layout{1, n_last});
  if (rc != TRIDIAG_OK) return rc;
  launches += g_last_launches;
  for (size_t jj = lv.size(); jj-- > 0;) {
    const LargeLevel& L = lv[jj];
    const bool first = jj == 0;
    const T* ia = first ? a : bufs[jj - 1].a;
    const T* ib = first ? b : bufs[jj - 1].b;
    const T* ic = first ? c : bufs[jj - 1].c;
    const T* id = first ? d : bufs[jj - 1].d;
    T* ox = first ? x : bufs[jj - 1].d;
    const bool last = jj + 1 == lv.size();
    const cudaError_t e = col_pass<T>(2, ia, ib, ic, id, ox, nullptr, nullptr, nullptr,
                                      bufs[jj].d, L.n, first ? nr : L.n, first ? es : S, S,
                                      last ? 1 : S, last ? n_last : 1, L.kin, c_pad, st);
    if (e != cudaSuccess) return (int)e;
    launches += 1;
  }
  g_last_launches = launches;
  return TRIDIAG_OK;
}

int strided_plan(int64_t n, int64_t S, int64_t es, int dtype, int algo, int switch_level,
                 int64_t bottom_n, int64_t m_validated, StridedPlan* P) {
  const int64_t np = pad_n(n);
  P->m = m_validated;
  const bool has_cr = algo == TRIDIAG_CR || is_hybrid(algo);
  if (es == 1) {  // rows (contiguous or pitched): the large-n row passes
    const int64_t bn = resolve_bottom_n(dtype, bottom_n);
    if (bn < 0) return TRIDIAG_ERR_BOTTOM_N;
    if (np <= bn || !has_cr) {
      if (np > tridiag_max_n(dtype, algo)) return TRIDIAG_ERR_N_TOO_LARGE;
      if (is_hybrid(algo) && switch_level == 0) P->m = auto_m(np, dtype, algo);
      if (is_hybrid(algo) && P->m > tridiag_max_switch_level(dtype, algo, np)) return TRIDIAG_ERR_SWITCH_LEVEL;
      P->kind = 0;
      return TRIDIAG_OK;
    }
    P->m = large_m(np, dtype, algo, switch_level, bn);
    if (P->m < 0) return TRIDIAG_ERR_SWITCH_LEVEL;
    if (!large_plan(np, dtype, P->m, bn, &P->lv, &P->n_last)) return TRIDIAG_ERR_SWITCH_LEVEL;
    P->kind = 1;
    return TRIDIAG_OK;
  }
  // interleaved columns
  const int64_t bc = resolve_col_bottom(dtype, bottom_n);
  if (bc < 0) return TRIDIAG_ERR_BOTTOM_N;
  if (np > col_onchip_max(dtype) && has_cr) {
    const int64_t m = col_m(np, dtype, algo, switch_level, bc, &P->lv, &P->n_last);
    if (m > 0) {
      P->m = m;
      P->kind = 2;
      return TRIDIAG_OK;
    }
  }
  // no pass plan (PCR / RD, an m beyond the reduced size, or n <= bottom):
  // the on-chip strided kernels
  if (np > tridiag_max_n(dtype, algo)) return TRIDIAG_ERR_N_TOO_LARGE;
  if (is_hybrid(algo)) {
    P->m = switch_level == 0 ? auto_m(np, dtype, algo) : switch_level;
    if (P->m > tridiag_max_switch_level(dtype, algo, np)) return TRIDIAG_ERR_SWITCH_LEVEL;
  }
  P->kind = 0;
  return TRIDIAG_OK;
}

}  // namespace

extern "C" {

int tridiag_abi_version(void) { return TRIDIAG_ABI_VERSION; }

int tridiag_last_launch_count(void) { return g_last_launches; }

const char* tridiag_last_kernel_name(int i) {
  if (i < 0 || i >= g_kernel_log_len) return nullptr;
  const char* name = nullptr;
  if (cudaFuncGetName(&name, g_kernel_log[i]) != cudaSuccess) {
    cudaGetLastError();
    return nullptr;
  }
  return name;
}

int64_t tridiag_phase_stamps_of(int launch, int64_t* out, int64_t cap) {
  if (launch < 0 || launch >= g_kernel_log_len || launch >= kMaxKernelLog) return 0;
  std::lock_guard<std::mutex> lk(g_stamp_mu);
  if (!g_stamp_dev[launch] || !out || cap <= 0) return 0;
  const int64_t len = std::min<int64_t>(cap, g_stamp_len[launch]);
  if (cudaMemcpy(out, g_stamp_dev[launch], len * sizeof(long long), cudaMemcpyDeviceToHost) != cudaSuccess)
    return 0;
  return len;
}

int64_t tridiag_phase_stamps(int64_t* out, int64_t cap) {
  return tridiag_phase_stamps_of(g_kernel_log_len - 1, out, cap);
}

const char* tridiag_status_string(int status) {
  switch (status) {
    case TRIDIAG_OK: return "ok";
    case TRIDIAG_ERR_NULL: return "null pointer argument";
    case TRIDIAG_ERR_N: return "n must be >= 1";
    case TRIDIAG_ERR_N_TOO_LARGE: return "n exceeds tridiag_max_n(dtype, algo)";
    case TRIDIAG_ERR_NUM_SYSTEMS: return "num_systems must be >= 0";
    case TRIDIAG_ERR_DTYPE: return "invalid dtype";
    case TRIDIAG_ERR_ALGO: return "invalid algo";
    case TRIDIAG_ERR_SWITCH_LEVEL: return "invalid switch_level for this algo/n/dtype";
    case TRIDIAG_ERR_OVERLAP: return "x overlaps an input (only x == d is allowed)";
    case TRIDIAG_ERR_WORKSPACE: return "workspace missing or too small";
    case TRIDIAG_ERR_STRIDE: return "invalid strides (need >= 1, one of them 1, non-overlapping)";
    case TRIDIAG_ERR_BOTTOM_N: return "invalid bottom_n for the large-n path";
  }
  if (status > 0) return cudaGetErrorString((cudaError_t)status);
  return "unknown status";
}

int tridiag_paper_cr(const void* a, const void* b, const void* c, const void* d, void* x,
                     int64_t n, int64_t num_systems, int dtype, int mode, tridiag_stream_t stream) {
  begin_call();
  if (num_systems != 0 && (!a || !b || !c || !d || !x)) return TRIDIAG_ERR_NULL;
  if (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64) return TRIDIAG_ERR_DTYPE;
  if (mode != 0 && mode != 1) return TRIDIAG_ERR_ALGO;
  if (n < 2 || !is_pow2(n)) return TRIDIAG_ERR_N;
  if (n > 1024) return TRIDIAG_ERR_N_TOO_LARGE;
  if (num_systems < 0 || num_systems > 0x7fffffffLL) return TRIDIAG_ERR_NUM_SYSTEMS;
  const size_t bytes = (size_t)num_systems * (size_t)n * elem_size(dtype);
  if (bytes > 0) {
    if (overlaps(x, a, bytes) || overlaps(x, b, bytes) || overlaps(x, c, bytes)) return TRIDIAG_ERR_OVERLAP;
    if (x != d && overlaps(x, d, bytes)) return TRIDIAG_ERR_OVERLAP;
  }
  if (num_systems == 0) return TRIDIAG_OK;
  cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
  const cudaError_t e =
      dtype == TRIDIAG_F32
          ? paper_cr<float>(static_cast<const float*>(a), static_cast<const float*>(b),
                            static_cast<const float*>(c), static_cast<const float*>(d),
                            static_cast<float*>(x), n, num_systems, mode, st)
          : paper_cr<double>(static_cast<const double*>(a), static_cast<const double*>(b),
                             static_cast<const double*>(c), static_cast<const double*>(d),
                             static_cast<double*>(x), n, num_systems, mode, st);
  return e == cudaSuccess ? TRIDIAG_OK : (int)e;
}

void tridiag_reload_knobs(void) {
  std::call_once(g_knobs_once, read_knobs);
  read_knobs();
}

int64_t tridiag_max_n(int dtype, int algo) {
  if (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64) return 0;
  switch (algo) {
    case TRIDIAG_CR:
    case TRIDIAG_CR_PCR:
    case TRIDIAG_CR_RD: return max_n_cr(dtype);
    case TRIDIAG_PCR:
    case TRIDIAG_RD: return max_inner_m(dtype);
    case TRIDIAG_RD_STONE: return dtype == TRIDIAG_F32 ? 512 : 256;  // one warp, registers only
  }
  return 0;
}

int64_t tridiag_max_switch_level(int dtype, int algo, int64_t n) {
  if (!is_hybrid(algo) || (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64)) return 0;
  if (n < 1 || pad_n(n) > max_n_cr(dtype)) return 0;
  return std::min<int64_t>(pad_n(n), max_inner_m(dtype));
}

int tridiag_auto_switch_level(int64_t n, int dtype, int algo) {
  if (!is_hybrid(algo) || (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64)) return 0;
  if (n < 1 || pad_n(n) > max_n_cr(dtype)) return 0;
  return auto_m(pad_n(n), dtype, algo);
}

int tridiag_solve_batched_strided(const void* a, const void* b, const void* c, const void* d,
                                  void* x, int64_t n, int64_t num_systems, int64_t elem_stride,
                                  int64_t sys_stride, int dtype, int algo, int switch_level,
                                  tridiag_stream_t stream) {
  begin_call();
  int64_t m = 0;
  const int v = validate(a, b, c, d, x, n, num_systems, dtype, algo, switch_level, &m,
                         elem_stride, sys_stride);
  if (v != TRIDIAG_OK) return v;
  return solve_device(a, b, c, d, x, n, num_systems, dtype, algo, m,
                      reinterpret_cast<cudaStream_t>(stream),
                      normalise_layout(n, num_systems, elem_stride, sys_stride));
}

int tridiag_solve_batched(const void* a, const void* b, const void* c, const void* d, void* x,
                          int64_t n, int64_t num_systems, int dtype, int algo, int switch_level,
                          tridiag_stream_t stream) {
  return tridiag_solve_batched_strided(a, b, c, d, x, n, num_systems, 1, n, dtype, algo,
                                       switch_level, stream);
}

int64_t tridiag_max_n_large(int dtype, int algo) {
  if (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64) return 0;
  if (algo == TRIDIAG_CR || is_hybrid(algo)) return int64_t(1) << 30;
  return tridiag_max_n(dtype, algo);
}

int64_t tridiag_large_chunk(int dtype) {
  if (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64) return 0;
  return large_chunk_n(dtype);
}

int64_t tridiag_large_workspace_bytes(int64_t n, int64_t num_systems, int dtype, int algo,
                                      int switch_level, int64_t bottom_n) {
  if (n < 1 || num_systems < 0 || (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64)) return -1;
  if (algo < TRIDIAG_CR || algo > TRIDIAG_RD_STONE) return -1;
  const int64_t np = pad_n(n);
  if (np > tridiag_max_n_large(dtype, algo)) return -1;
  const int64_t bn = resolve_bottom_n(dtype, bottom_n);
  if (bn < 0) return -1;
  if (np <= bn || !(algo == TRIDIAG_CR || is_hybrid(algo))) return 0;
  const int64_t m = large_m(np, dtype, algo, switch_level, bn);
  if (m < 0) return -1;
  std::vector<LargeLevel> lv;
  int64_t n_last = 0;
  if (!large_plan(np, dtype, m, bn, &lv, &n_last)) return -1;
  return (int64_t)large_ws_bytes(lv, num_systems, dtype);
}

int tridiag_solve_batched_large(const void* a, const void* b, const void* c, const void* d,
                                void* x, int64_t n, int64_t num_systems, int dtype, int algo,
                                int switch_level, int64_t bottom_n, void* workspace,
                                int64_t workspace_bytes, tridiag_stream_t stream) {
  begin_call();
  int64_t m = 0;
  const int v = validate(a, b, c, d, x, n, num_systems, dtype, algo, switch_level, &m, 1, n, true);
  if (v != TRIDIAG_OK) return v;
  const int64_t bn = resolve_bottom_n(dtype, bottom_n);
  if (bn < 0) return TRIDIAG_ERR_BOTTOM_N;
  const int64_t np = pad_n(n);
  cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
  if (np <= bn) {  // fits on chip: the plain entry point's path
    if (is_hybrid(algo) && switch_level == 0) m = auto_m(np, dtype, algo);
    if (is_hybrid(algo) && m > tridiag_max_switch_level(dtype, algo, np)) return TRIDIAG_ERR_SWITCH_LEVEL;
    return solve_device(a, b, c, d, x, n, num_systems, dtype, algo, m, st, Layout{1, n});
  }
  if (!(algo == TRIDIAG_CR || is_hybrid(algo))) return TRIDIAG_ERR_N_TOO_LARGE;
  m = large_m(np, dtype, algo, switch_level, bn);
  if (m < 0) return TRIDIAG_ERR_SWITCH_LEVEL;
  std::vector<LargeLevel> lv;
  int64_t n_last = 0;
  if (!large_plan(np, dtype, m, bn, &lv, &n_last)) return TRIDIAG_ERR_SWITCH_LEVEL;
  if (num_systems == 0) return TRIDIAG_OK;
  const size_t need = large_ws_bytes(lv, num_systems, dtype);
  if (!workspace || workspace_bytes < 0 || (size_t)workspace_bytes < need) return TRIDIAG_ERR_WORKSPACE;
  char* ws = static_cast<char*>(workspace);
  if (dtype == TRIDIAG_F32)
    return solve_large_t<float>(static_cast<const float*>(a), static_cast<const float*>(b),
                                static_cast<const float*>(c), static_cast<const float*>(d),
                                static_cast<float*>(x), n, num_systems, dtype, algo, m, lv, n_last,
                                ws, st, n);
  return solve_large_t<double>(static_cast<const double*>(a), static_cast<const double*>(b),
                               static_cast<const double*>(c), static_cast<const double*>(d),
                               static_cast<double*>(x), n, num_systems, dtype, algo, m, lv, n_last,
                               ws, st, n);
}

int64_t tridiag_column_chunk(int dtype) {
  if (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64) return 0;
  return col_chunk_n(dtype);
}

int64_t tridiag_strided_large_workspace_bytes(int64_t n, int64_t num_systems,
                                              int64_t elem_stride, int64_t sys_stride, int dtype,
                                              int algo, int switch_level, int64_t bottom_n) {
  if (n < 1 || num_systems < 0 || (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64)) return -1;
  if (algo < TRIDIAG_CR || algo > TRIDIAG_RD_STONE) return -1;
  if (elem_stride < 1 || sys_stride < 1) return -1;
  if (pad_n(n) > tridiag_max_n_large(dtype, algo)) return -1;
  elem_stride = normalise_layout(n, num_systems, elem_stride, sys_stride).es;
  StridedPlan P;
  if (strided_plan(n, num_systems, elem_stride, dtype, algo, switch_level, bottom_n, switch_level, &P) !=
      TRIDIAG_OK)
    return -1;
  if (P.kind == 1) return (int64_t)large_ws_bytes(P.lv, num_systems, dtype);
  if (P.kind == 2) return (int64_t)col_need(P, n, num_systems, dtype, algo, bottom_n);
  return 0;
}

int tridiag_solve_batched_strided_large(const void* a, const void* b, const void* c,
                                        const void* d, void* x, int64_t n, int64_t num_systems,
                                        int64_t elem_stride, int64_t sys_stride, int dtype,
                                        int algo, int switch_level, int64_t bottom_n,
                                        void* workspace, int64_t workspace_bytes,
                                        tridiag_stream_t stream) {
  begin_call();
  int64_t m = 0;
  const int v = validate(a, b, c, d, x, n, num_systems, dtype, algo, switch_level, &m, elem_stride,
                         sys_stride, true);
  if (v != TRIDIAG_OK) return v;
  {
    const Layout nl = normalise_layout(n, num_systems, elem_stride, sys_stride);
    elem_stride = nl.es;
    sys_stride = nl.ss;
  }
  StridedPlan P;
  const int pv = strided_plan(n, num_systems, elem_stride, dtype, algo, switch_level, bottom_n, m, &P);
  if (pv != TRIDIAG_OK) return pv;
  cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
  if (P.kind == 0)
    return solve_device(a, b, c, d, x, n, num_systems, dtype, algo, P.m, st,
                        Layout{elem_stride, sys_stride});
  if (num_systems == 0) return TRIDIAG_OK;
  const size_t need = P.kind == 1 ? large_ws_bytes(P.lv, num_systems, dtype)
                                  : col_need(P, n, num_systems, dtype, algo, bottom_n);
  if (!workspace || workspace_bytes < 0 || (size_t)workspace_bytes < need) return TRIDIAG_ERR_WORKSPACE;
  char* ws = static_cast<char*>(workspace);
  if (P.kind == 1) {
    if (dtype == TRIDIAG_F32)
      return solve_large_t<float>(static_cast<const float*>(a), static_cast<const float*>(b),
                                  static_cast<const float*>(c), static_cast<const float*>(d),
                                  static_cast<float*>(x), n, num_systems, dtype, algo, P.m, P.lv,
                                  P.n_last, ws, st, num_systems > 1 ? sys_stride : n);
    return solve_large_t<double>(static_cast<const double*>(a), static_cast<const double*>(b),
                                 static_cast<const double*>(c), static_cast<const double*>(d),
                                 static_cast<double*>(x), n, num_systems, dtype, algo, P.m, P.lv,
                                 P.n_last, ws, st, num_systems > 1 ? sys_stride : n);
  }
  if (dtype == TRIDIAG_F32)
    return solve_col_t<float>(static_cast<const float*>(a), static_cast<const float*>(b),
                              static_cast<const float*>(c), static_cast<const float*>(d),
                              static_cast<float*>(x), n, num_systems, elem_stride, dtype, algo, P.m,
                              P.lv, P.n_last, ws, st);
  return solve_col_t<double>(static_cast<const double*>(a), static_cast<const double*>(b),
                             static_cast<const double*>(c), static_cast<const double*>(d),
                             static_cast<double*>(x), n, num_systems, elem_stride, dtype, algo, P.m,
                             P.lv, P.n_last, ws, st);
}

// Host pipeline depth: three chunk buffers on three streams, so the
// host-to-device engine can run ahead of a device-to-host copy that still
// occupies the previous buffer.
constexpr int kHostBufs = 3;

size_t tridiag_host_workspace_bytes(int64_t n, int dtype, int64_t chunk_systems) {
  if (n < 1 || chunk_systems < 0 || (dtype != TRIDIAG_F32 && dtype != TRIDIAG_F64)) return 0;
  if (chunk_systems == 0) chunk_systems = std::max<int64_t>(1, (int64_t(16) << 20) / (4 * n * (int64_t)elem_size(dtype)));
  return (size_t)kHostBufs * 4 * (size_t)chunk_systems * (size_t)n * elem_size(dtype);
}

int tridiag_solve_batched_host(const void* a, const void* b, const void* c, const void* d, void* x,
                               int64_t n, int64_t num_systems, int dtype, int algo,
                               int switch_level, void* workspace, size_t workspace_bytes,
                               int64_t chunk_systems) {
  begin_call();
  int64_t m = 0;
  const int v = validate(a, b, c, d, x, n, num_systems, dtype, algo, switch_level, &m, 1, n);
  if (v != TRIDIAG_OK) return v;
  if (num_systems == 0) return TRIDIAG_OK;
  if (chunk_systems < 0) return TRIDIAG_ERR_NUM_SYSTEMS;
  if (chunk_systems == 0)
    chunk_systems = std::max<int64_t>(1, (int64_t(16) << 20) / (4 * n * (int64_t)elem_size(dtype)));
  chunk_systems = std::min<int64_t>(chunk_systems, num_systems);
  const size_t need = tridiag_host_workspace_bytes(n, dtype, chunk_systems);
  if (!workspace || workspace_bytes < need) return TRIDIAG_ERR_WORKSPACE;

  const size_t T = elem_size(dtype);
  const size_t arr = (size_t)chunk_systems * (size_t)n * T;  // one array of one chunk
  cudaStream_t st[kHostBufs];
  for (int i = 0; i < kHostBufs; ++i) {
    if (cudaStreamCreateWithFlags(&st[i], cudaStreamNonBlocking) != cudaSuccess) {
      for (int j = 0; j < i; ++j) cudaStreamDestroy(st[j]);
      return (int)cudaGetLastError();
    }
  }
  // The workspace may have been handed out by a caching allocator while work
  // queued earlier on the legacy default stream (which orders every blocking
  // stream) still uses it: the internal streams wait for that work first.
  {
    cudaEvent_t ev;
    if (cudaEventCreateWithFlags(&ev, cudaEventDisableTiming) != cudaSuccess ||
        cudaEventRecord(ev, cudaStreamLegacy) != cudaSuccess) {
      for (int i = 0; i < kHostBufs; ++i) cudaStreamDestroy(st[i]);
      return (int)cudaGetLastError();
    }
    for (int i = 0; i < kHostBufs; ++i) cudaStreamWaitEvent(st[i], ev, 0);
    cudaEventDestroy(ev);
  }
  int rc = TRIDIAG_OK;
  int launches = 0;
  const char* hp[4] = {static_cast<const char*>(a), static_cast<const char*>(b),
                       static_cast<const char*>(c), static_cast<const char*>(d)};
  char* hx = static_cast<char*>(x);
  for (int64_t s0 = 0, j = 0; s0 < num_systems && rc == TRIDIAG_OK; s0 += chunk_systems, ++j) {
    const int64_t cnt = std::min<int64_t>(chunk_systems, num_systems - s0);
    const size_t bytes = (size_t)cnt * (size_t)n * T;
    const size_t off = (size_t)s0 * (size_t)n * T;
    cudaStream_t s = st[j % kHostBufs];
    char* buf = static_cast<char*>(workspace) + (size_t)(j % kHostBufs) * 4 * arr;
    for (int q = 0; q < 4; ++q) {
      cudaError_t e = cudaMemcpyAsync(buf + q * arr, hp[q] + off, bytes, cudaMemcpyHostToDevice, s);
      if (e != cudaSuccess) { rc = (int)e; break; }
    }
    if (rc != TRIDIAG_OK) break;
    // x overwrites the chunk's d in place on the device.
    rc = solve_device(buf, buf + arr, buf + 2 * arr, buf + 3 * arr, buf + 3 * arr, n, cnt, dtype,
                      algo, m, s, Layout{1, n});
    launches += g_last_launches;
    if (rc != TRIDIAG_OK) break;
    cudaError_t e = cudaMemcpyAsync(hx + off, buf + 3 * arr, bytes, cudaMemcpyDeviceToHost, s);
    if (e != cudaSuccess) rc = (int)e;
  }
  for (int i = 0; i < kHostBufs; ++i) {
    const cudaError_t e = cudaStreamSynchronize(st[i]);
    if (rc == TRIDIAG_OK && e != cudaSuccess) rc = (int)e;
    cudaStreamDestroy(st[i]);
  }
  g_last_launches = launches;
  return rc;
}

}  // extern "C"

/*
 * tridiag.h -- C ABI of libtridiag.so, the B200 (sm_100a) batched tridiagonal
 * solver library.
 *
 * Method: Zhang, Cohen, Owens, "Fast Tridiagonal Solvers on the GPU",
 * PPoPP'10 (/root/reference/PAPER.md, cited P:L<line>).  The library solves a
 * batch of independent tridiagonal systems ("solving a large
 * number of small tridiagonal systems in parallel") with cyclic reduction
 * (CR, section 2.1), parallel cyclic reduction (PCR, section 2.2
 * P:L313-386), recursive doubling (RD, section 2.3) or the hybrids
 * CR+PCR and CR+RD (section 3, Fig 4).
 *
 * No torch or CUDA types appear in this header; `tridiag_stream_t` is
 * ABI-identical to cudaStream_t / CUstream.
 */
#ifndef TRIDIAG_H_
#define TRIDIAG_H_

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define TRIDIAG_ABI_VERSION 1

typedef struct CUstream_st* tridiag_stream_t; /* == cudaStream_t; NULL = legacy default stream */

/* Element type of all five arrays. */
typedef enum { TRIDIAG_F32 = 0, TRIDIAG_F64 = 1 } tridiag_dtype;

/* Algorithm.  The hybrids take an intermediate system size m (switch_level). */
typedef enum {
    TRIDIAG_CR = 0,     /* P:L272-312, Fig 1                                    */
    TRIDIAG_PCR = 1,    /* P:L313-386, Fig 2                                    */
    TRIDIAG_RD = 2,     /* P:L387-421, Fig 3 (Egecioglu scan form of Stone's RD) */
    TRIDIAG_CR_PCR = 3, /* P:L572-581, Fig 4: CR to m equations, PCR, CR back   */
    TRIDIAG_CR_RD = 4,  /* P:L572-581, Fig 4: CR to m equations, RD, CR back    */
    /* Not one of the paper's five: overflow-free recursive doubling in LU
     * form (the paper's RD overflows on dominant rows,
     * P:L1219-1236, and it cites Stone [27]): three Hillis-Steele scans --
     * power-of-two-rescaled 2x2 continuant products for the LU pivots, then
     * the forward and backward affine recurrences, which contract on
     * diagonally dominant rows.  n <= 512 (fp32) / 256 (fp64). */
    TRIDIAG_RD_STONE = 5
} tridiag_algo;

/* Status codes.  0 = enqueued.  Negative = argument error, nothing enqueued.
 * Positive = the cudaError_t reported by the runtime. */
enum {
    TRIDIAG_OK = 0,
    TRIDIAG_ERR_NULL = -1,         /* a pointer is NULL while num_systems > 0        */
    TRIDIAG_ERR_N = -2,            /* n < 1                                          */
    TRIDIAG_ERR_N_TOO_LARGE = -3,  /* next power of two of n > tridiag_max_n         */
    TRIDIAG_ERR_NUM_SYSTEMS = -4,  /* num_systems < 0                                */
    TRIDIAG_ERR_DTYPE = -5,        /* dtype not a tridiag_dtype                      */
    TRIDIAG_ERR_ALGO = -6,         /* algo not a tridiag_algo                        */
    TRIDIAG_ERR_SWITCH_LEVEL = -7, /* invalid switch_level for this algo / n / dtype */
    TRIDIAG_ERR_OVERLAP = -8,      /* x overlaps an input other than exactly x == d  */
    TRIDIAG_ERR_WORKSPACE = -9,    /* host entry point: workspace too small / NULL   */
    TRIDIAG_ERR_STRIDE = -10,      /* strided entry point: invalid strides           */
    TRIDIAG_ERR_BOTTOM_N = -11     /* large-n entry point: invalid bottom_n          */
};

/*
 * tridiag_solve_batched -- solve num_systems independent systems on the GPU.
 *
 * For every s in [0, num_systems) and i in [0, n):
 *     a[s*n+i] x[s*n+i-1] + b[s*n+i] x[s*n+i] + c[s*n+i] x[s*n+i+1] = d[s*n+i]
 * with x_{-1} = x_n = 0.  a[s*n] and c[s*n+n-1] are NOT matrix
 * entries (the paper's matrix has no a_1 and no c_n) and are never read as
 * coefficients: any value, including NaN, is allowed there.
 *
 * Layout: five device arrays of S*n elements of `dtype`,
 * system-major ("the data of the first system stored at the beginning of the
 * arrays, followed by the second system, ...").
 *
 * a, b, c, d  device pointers, read only.
 * x           device pointer, written.  x == d (exact in-place) is allowed;
 *             any other overlap of x with an input is TRIDIAG_ERR_OVERLAP.
 * n           equations per system, n >= 1.  The paper's solvers take powers of
 *             two; other n are solved as the next power of two
 *             n_pad with padding equations x_i + c_pad x_{i+1} = 0 (i >= n,
 *             solution 0; c_pad = 1 for the RD inner, which needs nonzero
 *             c, else 0) and only the n real elements are read / written
 *             (scalar-load path).  n_pad <= tridiag_max_n(dtype, algo).
 * num_systems S >= 0.  S == 0 returns TRIDIAG_OK without launching (the
 *             pointers may then be NULL; the other arguments are validated).
 * dtype       TRIDIAG_F32 or TRIDIAG_F64.  All arithmetic is in this type.
 * algo        tridiag_algo.
 * switch_level  the intermediate system size m of the hybrids (Fig 17's
 *             x-axis, "size-256 intermediate"): 0 = the tuned
 *             table (tridiag_auto_switch_level); else a power of two with
 *             2 <= m <= n_pad and m <= tridiag_max_switch_level(dtype, algo, n).
 *             m = 2 reproduces CR and m = n reproduces PCR / RD.  Must be 0
 *             for the non-hybrid algorithms.
 * stream      CUDA stream the work is enqueued on (asynchronous, no host
 *             synchronisation).
 *
 * Pointers must be device memory of the current device.  Alignment: the
 * vector path needs every pointer aligned to the per-thread tile
 * (min(32, R*sizeof(T)) bytes); ragged n with n*sizeof(T) a multiple of 16
 * and 16-byte aligned pointers takes 16-byte / TMA vector paths; otherwise a
 * staged scalar-load path runs (bitwise the same results in every case).
 * Launches carry the programmatic-dependent-launch attribute: a kernel's
 * thread blocks may be scheduled while the previous work on the stream
 * drains, but every kernel waits for it (griddepcontrol.wait) before its
 * first memory access, so stream order is unchanged.  Results are deterministic: bitwise identical across runs and
 * across any partitioning of the batch.  Numeric failure (a zero pivot; RD
 * overflow outside its stable regime) is not an error code: it
 * shows up as non-finite x (no pivoting).
 *
 * Thread safety: reentrant; the only global state is immutable tables and a
 * per-device launch-configuration cache built under a lock.
 */
int tridiag_solve_batched(const void* a, const void* b, const void* c, const void* d,
                          void* x, int64_t n, int64_t num_systems, int dtype, int algo,
                          int switch_level, tridiag_stream_t stream);

/*
 * tridiag_solve_batched_strided -- the same solve for strided layouts
 * (SURVEY.md 8(f) NEXT f1): element i of system s of every array is at
 * ptr[s * sys_stride + i * elem_stride] (strides in elements, >= 1, one of
 * them 1, the mapping one-to-one: sys_stride >= elem_stride * n or
 * elem_stride >= sys_stride * num_systems).  (1, n) is the contiguous layout
 * of tridiag_solve_batched; (1, pitch) a pitched row sweep; (es, 1) with
 * es >= num_systems is the ADI column sweep of a row-major grid ("the most
 * common application", ADI): e.g. the columns of an
 * NY x NX grid are NX systems of n = NY with elem_stride = NX, sys_stride = 1.
 * Interleaved layouts are staged through shared memory in tiles of 8-32
 * consecutive systems (coalesced row segments); pitched rows whose pitch is
 * a multiple of 16 bytes take the same vector paths as contiguous rows;
 * other non-contiguous layouts use scalar loads.  x must use the same
 * strides; x == d is allowed.
 * Errors as tridiag_solve_batched plus TRIDIAG_ERR_STRIDE.
 */
int tridiag_solve_batched_strided(const void* a, const void* b, const void* c, const void* d,
                                  void* x, int64_t n, int64_t num_systems, int64_t elem_stride,
                                  int64_t sys_stride, int dtype, int algo, int switch_level,
                                  tridiag_stream_t stream);

/*
 * tridiag_solve_batched_host -- the same solve for HOST arrays (the paper's
 * "with transfer" case).  a, b, c, d, x are host pointers
 * (pinned memory gives full-speed asynchronous copies; pageable memory works
 * but serialises).  The batch is split into chunks that are pipelined over
 * three CUDA streams / buffers: host-to-device copies of the next chunks and
 * the device-to-host copy of earlier ones overlap the solve of chunk j.
 *
 * workspace        device buffer owned by the caller, at least
 *                  tridiag_host_workspace_bytes(n, dtype, chunk_systems) bytes.
 * chunk_systems    systems per chunk (> 0; 0 = library default).
 * The call BLOCKS until x is written (it is a host-memory API).
 * x == d is allowed; other overlaps are TRIDIAG_ERR_OVERLAP.
 */
int tridiag_solve_batched_host(const void* a, const void* b, const void* c, const void* d,
                               void* x, int64_t n, int64_t num_systems, int dtype, int algo,
                               int switch_level, void* workspace, size_t workspace_bytes,
                               int64_t chunk_systems);
size_t tridiag_host_workspace_bytes(int64_t n, int dtype, int64_t chunk_systems);

/*
 * tridiag_solve_batched_large -- systems larger than tridiag_max_n (SURVEY.md
 * 8(f) NEXT f2; "accelerate larger systems with several first steps (as in
 * CR) that reduce the system to fit into shared memory").
 *
 * Same arguments, semantics, layout (contiguous, system stride n) and errors
 * as tridiag_solve_batched, for CR, CR+PCR and CR+RD with
 * n_pad <= tridiag_max_n_large(dtype, algo) (2^30).  PCR, RD and RD_STONE
 * have no CR levels to reduce with: for them (and for any n_pad <= bottom_n)
 * this is exactly tridiag_solve_batched.
 *
 * Method: passes of log2 R CR levels (R = 16 fp32 / 8 fp64 equations per
 * lane; chunks of tridiag_large_chunk(dtype) equations per CTA) write the
 * surviving n / R equations of every system to the workspace, until the
 * system has at most bottom_n equations; the on-chip kernels solve it (CR,
 * or the hybrid with intermediate size m); expansion passes recompute each
 * level's forward steps from its input and back-substitute.  Every equation
 * update is the same correctly rounded operation sequence as in the on-chip
 * kernels, so CR and CR+PCR results are bitwise identical to
 * tridiag_solve_batched wherever both apply.  HBM traffic is about
 * 10 n T bytes per system (each level read twice) against 5 n T on chip.
 *
 * switch_level  hybrids: 0 = the tuned m of the size the passes reduce to;
 *             else a power of two m with 2 <= m <= tridiag_max_switch_level
 *             at that size (m caps the CR levels: the passes stop at m).
 * bottom_n    largest system solved on chip; 0 = tridiag_max_n(dtype, CR),
 *             else a power of two in [tridiag_large_chunk(dtype) / 2,
 *             tridiag_max_n(dtype, CR)] (TRIDIAG_ERR_BOTTOM_N otherwise).
 * workspace   device buffer owned by the caller, >= tridiag_large_workspace_bytes
 *             bytes (256-byte aligned for the vector path; NULL allowed when
 *             that is 0).  Holds the reduced systems (4 arrays per level, the
 *             deepest one solved in place); about 4 S n T / (R - 1) bytes.
 * Asynchronous on `stream` like tridiag_solve_batched; x == d allowed.
 */
int tridiag_solve_batched_large(const void* a, const void* b, const void* c, const void* d,
                                void* x, int64_t n, int64_t num_systems, int dtype, int algo,
                                int switch_level, int64_t bottom_n, void* workspace,
                                int64_t workspace_bytes, tridiag_stream_t stream);
/* Workspace bytes tridiag_solve_batched_large needs (0 when n fits on chip);
 * -1 for invalid arguments. */
int64_t tridiag_large_workspace_bytes(int64_t n, int64_t num_systems, int dtype, int algo,
                                      int switch_level, int64_t bottom_n);
/* Largest n of tridiag_solve_batched_large for (dtype, algo); 0 if invalid. */
int64_t tridiag_max_n_large(int dtype, int algo);
/* Equations per reduction chunk (one CTA) of the large-n passes. */
int64_t tridiag_large_chunk(int dtype);

/*
 * tridiag_solve_batched_strided_large -- tridiag_solve_batched_strided with a
 * workspace, for strided layouts whose systems do not fit one CTA's on-chip
 * kernel in that layout (SURVEY.md 8(f) NEXT f1 + f2).  Same arguments,
 * layout rules (element (s, i) at ptr[s * sys_stride + i * elem_stride]),
 * semantics and errors as tridiag_solve_batched_strided, plus bottom_n /
 * workspace as in tridiag_solve_batched_large; n_pad up to
 * tridiag_max_n_large for CR and the hybrids.
 *
 * Rows (elem_stride == 1, contiguous or pitched): exactly
 * tridiag_solve_batched_large (row reduction passes while n_pad > bottom_n).
 *
 * Interleaved columns (sys_stride == 1, elem_stride >= num_systems: the ADI
 * column sweep): for CR, CR+PCR and CR+RD with
 * n_pad > 32 R (512 fp32 / 256 fp64, the on-chip interleaved kernel's
 * capacity), column reduction passes of log2 R CR levels -- one
 * CTA per 32 consecutive systems x W R rows, every warp access one coalesced
 * row segment of 32 systems -- at least one, then more until at most
 * bottom_n equations remain; the last pass writes the surviving equations
 * TRANSPOSED into contiguous rows of the workspace, which the row kernels
 * solve (the same kernels as tridiag_solve_batched); expansion passes
 * back-substitute and write x.  bottom_n: 0 = tridiag_max_n
 * (one pass for every on-chip size), else a power of two in
 * [tridiag_column_chunk(dtype) / 2, tridiag_max_n(dtype, CR)].  HBM traffic
 * about 9.3 n T per system (the input is read twice) against 5 n T on chip,
 * but every access is a full row segment where the on-chip strided kernel
 * reads 4-byte pieces of 32-byte sectors.  Hybrid default m: the contiguous
 * solve's tuned m of the full size, so results are bitwise identical to
 * tridiag_solve_batched on the transposed data.  PCR, RD, RD_STONE, and
 * hybrid m that the passes cannot reach, take the on-chip strided path
 * (no workspace).
 *
 * workspace   caller-owned device buffer of at least
 *             tridiag_strided_large_workspace_bytes(...) bytes (0 when no
 *             passes run; NULL allowed then); 256-byte aligned.
 * Asynchronous on `stream`; x == d allowed.
 */
int tridiag_solve_batched_strided_large(const void* a, const void* b, const void* c,
                                        const void* d, void* x, int64_t n, int64_t num_systems,
                                        int64_t elem_stride, int64_t sys_stride, int dtype,
                                        int algo, int switch_level, int64_t bottom_n,
                                        void* workspace, int64_t workspace_bytes,
                                        tridiag_stream_t stream);
/* Workspace bytes of tridiag_solve_batched_strided_large; -1 if invalid. */
int64_t tridiag_strided_large_workspace_bytes(int64_t n, int64_t num_systems,
                                              int64_t elem_stride, int64_t sys_stride, int dtype,
                                              int algo, int switch_level, int64_t bottom_n);
/* Rows per column-pass chunk (one CTA: W R rows of 32 systems). */
int64_t tridiag_column_chunk(int dtype);

/* Human-readable text of a status code (static storage, never NULL). */
const char* tridiag_status_string(int status);

/* Largest n this build solves for (dtype, algo); 0 for invalid arguments. */
int64_t tridiag_max_n(int dtype, int algo);

/* Largest legal intermediate size m for a hybrid at this (dtype, n); for
 * the non-hybrids 0.  Bounded by the on-chip capacity of the inner solver. */
int64_t tridiag_max_switch_level(int dtype, int algo, int64_t n);

/* The tuned intermediate size m used when switch_level == 0 (hybrids), from
 * the switch-level sweep compiled into the library; 0 for non-hybrids or
 * invalid arguments. */
int tridiag_auto_switch_level(int64_t n, int dtype, int algo);

/*
 * tridiag_paper_cr -- BASELINE ONLY, not a solver to use: the paper's own
 * GT200 kernel schedule for CR (one CTA per system, n/2 threads,
 * the system in place in shared memory, a __syncthreads per step, the access
 * stride doubling every step), kept so its bank conflicts and per-step times
 * (Fig 9) can be measured on B200 beside the register-blocked
 * kernels.  Same layout, ownership and stream semantics as
 * tridiag_solve_batched (contiguous, x == d allowed); n a power of two,
 * 2 <= n <= 1024; num_systems <= 2^31 - 1 (one CTA per system).
 * mode 0: the schedule as published (correct x, G1/G2 accuracy).
 * mode 1: the paper's timing control, every access at stride
 *         one -- x is MEANINGLESS, for timing / ncu comparison only.
 * With TRIDIAG_PHASE_STAMPS=1, thread 0 of each of the first 512 CTAs records
 * clock64() after the load, each forward step, the 2x2 solve, each backward
 * step and the store (32 slots per CTA; tridiag_phase_stamps).
 * Returns the same status codes (mode outside {0, 1}: TRIDIAG_ERR_ALGO).
 */
int tridiag_paper_cr(const void* a, const void* b, const void* c, const void* d, void* x,
                     int64_t n, int64_t num_systems, int dtype, int mode,
                     tridiag_stream_t stream);

/* Re-read the TRIDIAG_* tuning knobs from the environment (diagnostic: A/B
 * measurements and the bitwise path-equality tests).  Normally the knobs are
 * read once, on the library's first call, and never change afterwards; calling
 * this while another thread is solving is allowed (each knob is an atomic) but
 * that solve may see either value.  No effect on results except which of
 * several bitwise-equal kernels runs. */
void tridiag_reload_knobs(void);

/* TRIDIAG_ABI_VERSION of the loaded library. */
int tridiag_abi_version(void);

/* Number of kernel launches the last successful tridiag_solve_batched call
 * made on this thread (0 when S == 0).  For the bench's launch count. */
int tridiag_last_launch_count(void);

/* Name (the mangled device-function symbol, as ncu prints it with
 * --print-kernel-base mangled) of the i-th kernel launched by the last call
 * on this thread, i = 0 .. min(tridiag_last_launch_count(), 16) - 1; NULL
 * otherwise.  Static storage owned by the CUDA runtime.  Diagnostic: lets a
 * benchmark name the kernel it timed and look up its profile. */
const char* tridiag_last_kernel_name(int i);

/*
 * tridiag_phase_stamps -- diagnostic (the analogue of
 * the paper's per-phase timing, Figs 8/11/13/15/16).  Only active
 * when the process runs with TRIDIAG_PHASE_STAMPS=1: the warp kernels then
 * record clock64() on lane 0 of warp 0 of every CTA at the phase boundaries
 * of its first 4 system groups, as rows of 8 int64:
 *   [0] start  [1] loads + in-lane CR forward  [2] tail chain
 *   [3] lane-level CR + inner PCR/RD (or blocked inner)
 *   [4] in-lane back-substitution  [5] store issued  [6..7] unused (0)
 * The TMA CTA kernel (n > 32 R) records, on warp 0:
 *   [0] wait for the stage  [1] data arrived  [2] in-lane forward + next-warp
 *   heads  [3] lane-level forward  [4] survivors solved  [5] lane-level
 *   back-substitution  [6] in-lane back-substitution  [7] store issued
 * (RD inner: [3], [4] stay 0).  The column passes: reduce [0] unit start
 * [1] stage arrived [2] in-lane forward [3] heads + tail chain [4] survivors
 * stored; expand [0] start [1] x2 + stage [2] forward recomputed [3] back-
 * substituted [4] stored.  The large-n passes: reduce [0] start [1] loads +
 * forward [2] survivors stored; expand [0] start [1] loads + forward [2]
 * back-substituted [3] stored.  One row of 8 per CTA per unit (first 4).
 * tridiag_paper_cr: 32 slots per CTA (see there).
 * Copies up to `cap` values of the last launch of the last call on this
 * thread into host `out` (synchronous) and returns how many; 0 when inactive.
 */
int64_t tridiag_phase_stamps(int64_t* out, int64_t cap);
/* The same for launch `launch` (0-based, < 16) of the last call on this
 * thread (multi-launch calls: the large-n and column passes). */
int64_t tridiag_phase_stamps_of(int launch, int64_t* out, int64_t cap);

#ifdef __cplusplus
}
#endif
#endif /* TRIDIAG_H_ */

/*
 * tds.h -- C ABI of libtds, the B200-native multi-stage batched tridiagonal
 * solver (Davidson, Zhang & Owens, "An Auto-tuned Method for Solving Large
 * Tridiagonal Systems on the GPU", IPDPS 2011).  "P:Lx" = line x of the
 * paper's text; "§8" = SURVEY.md §8, the hot-path contract.
 *
 * WHAT IS SOLVED.  m independent tridiagonal systems of n equations
 *        a_i x_{i-1} + b_i x_i + c_i x_{i+1} = d_i,   i = 0..n-1
 * ("tridiagonal systems of any size and number, as long as they fit into
 * global memory"; the workload [m, n] of Fig. 1).
 * a_0 and c_{n-1} of every system are ignored (treated as 0).
 *
 * HOW (the paper's four stages in sm_100a kernels, §III):
 *   stages 1+2  k global PCR splitting levels in
 *               one or more fused HBM passes -> 2^k interleaved subsystems;
 *   stages 3+4  each subsystem solved on-chip by the hybrid kernel: c CR
 *               levels in registers, PCR on the reduced system until T
 *               independent chains, Thomas per chain, CR back substitution
 *               (base kernel §III-A; switch points §III-D).
 * The switch points come from one of the paper's three parameter-selection
 * methods (§IV): DEFAULT (machine-oblivious), STATIC (device
 * query) or TUNED (self-tuned from the static seed, tds_tune).
 *
 * NUMERICS.  No pivoting (the paper's solvers do not pivot): the precondition
 * is a nonsingular, diagonally dominant (or SPD) system.  Breakdown is NOT
 * detected: a zero pivot yields inf/NaN in x.  fp32 uses the hardware
 * approximate reciprocal (rcp.approx, <= 1 ulp); fp64 uses the hardware
 * reciprocal seed refined by two Newton steps (~1 ulp) -- DESIGN.md R16.
 *
 * CONVENTIONS (every entry point):
 *  - Layout: element i of system s is at ptr[s * batch_stride + i]
 *    (system-major; batch_stride >= n; batch_stride == 0 means n).
 *  - Device pointers are caller-owned device memory of the plan's dtype,
 *    aligned to sizeof(T).  Host pointers are documented as such.
 *  - Plans are host objects and own NO device memory.  A plan is immutable
 *    except through tds_tune / tds_plan_set_params; concurrent solves with one
 *    plan on different streams need separate workspaces.
 *  - Streams: a cudaStream_t passed as void* (NULL = legacy default stream).
 *    Solve entry points only enqueue work and return (asynchronous).
 *  - Errors: every call returns tds_status; no exception crosses the ABI.
 *    Argument errors are detected before anything is enqueued.  Launch
 *    failures return TDS_ERR_CUDA.  tds_last_error() gives a thread-local
 *    human-readable detail for the most recent failing call.
 */
#ifndef TDS_H_
#define TDS_H_

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define TDS_VERSION 100 /* 1.0.0 */
#define TDS_MAX_PASSES 8

typedef enum {
    TDS_OK = 0,
    TDS_ERR_INVALID_ARG = 1,     /* bad pointer, size, stride, mode, overlap      */
    TDS_ERR_UNSUPPORTED = 2,     /* valid request the kernels cannot run          */
    TDS_ERR_NO_MEMORY = 3,       /* host or device allocation failed              */
    TDS_ERR_WORKSPACE = 4,       /* workspace NULL / too small / misaligned       */
    TDS_ERR_CUDA = 5,            /* CUDA runtime or launch error                  */
    TDS_ERR_TUNE = 6,            /* tuner failed (trial error, cache I/O)         */
    TDS_ERR_DEVICE_MISMATCH = 7  /* current device differs from the plan's device */
} tds_status;

typedef enum { TDS_F32 = 0, TDS_F64 = 1 } tds_dtype;

/* Parameter-selection methods of §IV. */
typedef enum {
    TDS_PARAMS_DEFAULT = 0, /* §IV-B: 256-element on-chip entry, 16 systems, T = 32 */
    TDS_PARAMS_STATIC = 1,  /* §IV-C: device-query seeds (smem size, SM count, 2x warp) */
    TDS_PARAMS_TUNED = 2    /* §IV-D: set by tds_tune only (not accepted by tds_plan) */
} tds_param_mode;

typedef struct tds_plan_st *tds_plan_t;

/* Queryable device properties used by the planner (Table II). */
typedef struct {
    int32_t sm_count;              /* "Processors"                               */
    int32_t smem_optin_bytes;      /* max dynamic shared memory per block        */
    int32_t smem_per_sm_bytes;     /* "Shared Memory" per processor              */
    int32_t regs_per_sm;           /* "Register Memory"                          */
    int32_t max_threads_per_block;
    int32_t warp_size;
    int32_t cc_major, cc_minor;
    int64_t l2_bytes;
    int64_t global_mem_bytes;      /* "Global Mem"                               */
} tds_device_props;

/* The tunable integers of a plan (the switch points of §III-D). */
typedef struct {
    int32_t k;                       /* total split levels: 2^k subsystems per system   */
    int32_t passes;                  /* HBM split passes (0 iff k == 0)                 */
    int32_t k_pass[TDS_MAX_PASSES];  /* levels fused in each pass, sum == k             */
    int32_t cr_levels;               /* c: CR levels in registers (R = 2^c rows/thread)  */
    int32_t thomas_chains;           /* T: Thomas chains of the reduced system (pow2)   */
    int32_t cluster;                 /* CTAs (SMs) sharing one subsystem: 1,2,4,8,16    */
    int32_t tl_levels;               /* c2: CR levels across threads (shared memory)    */
    int32_t split_tile_rows;         /* shared-memory split pass tile (k_pass > 4 only) */
    int32_t split_threads;           /* shared-memory split pass CTA size (k_pass > 4)  */
    int32_t theta;                   /* stage 1->2 switch: independent systems needed   */
    int32_t chunk_systems;           /* systems per L2-resident chunk (0 = all at once) */
    int32_t split_only;              /* 1: plan only the split passes (tds_split_batched;
                                        on-chip limits not checked, tds_solve_* refuse) */
    int32_t x_group;                 /* 0: x placed by a separate kernel (k > 0).  G = 2, 4
                                        or 8: a cluster of G on-chip CTAs solves G adjacent
                                        residue classes (Fig. 3a) and stores x
                                        straight to rows r + 2^k j in G-element runs; needs
                                        k > 0, 2^k | n, G <= 2^k, one subsystem per CTA
                                        (n / 2^k = threads x 2^c), tl_levels = 5,
                                        2^c sizeof(T) = 64, G sizeof(T) >= 16, and
                                        2^k sizeof(T), batch_stride sizeof(T) multiples of 16 */
    int32_t strided;                 /* 1: the paper's strided base-kernel variant:
                                        the split leaves the 2^k subsystems interleaved in
                                        place (rows in original order) and the on-chip kernel
                                        gathers residue class r with stride 2^k and scatters x
                                        in place (no de-interleave, no placement kernel); needs
                                        one split pass with k_pass <= 4, cluster 1,
                                        tl_levels 5, 2^c sizeof(T) = 64, x_group 0.
                                        2: the paper's second variant, coalesced loads with a
                                        global-memory fallback: the same in-place
                                        split output; one CTA solves G = 32 / sizeof(T)
                                        consecutive residues (every access a whole 32-byte
                                        sector), holds as many of their rows as fit in shared
                                        memory and keeps the rest in the workspace, runs
                                        log2(thomas_chains) PCR levels and Thomas per chain,
                                        x stored in place; needs one split pass with
                                        log2(G) <= k_pass <= 4, cr_levels 0, tl_levels 0,
                                        cluster 1, x_group 0, G x thomas_chains <= 1024,
                                        batch_stride x sizeof(T) a multiple of 16;
                                        any subsystem length (no on-chip size limit) */
} tds_params;

/* Everything a plan decided (read-only view). */
typedef struct {
    int32_t dtype, mode, tuned;
    int32_t device;
    int64_t n, m, batch_stride;
    tds_params params;
    int64_t n_sub;            /* longest subsystem: ceil(n / 2^k)                      */
    int64_t num_subsystems;   /* m * min(2^k, n)                                       */
    int32_t n_sub_target;     /* stage 2->3 switch (subsystem size) the plan aimed at  */
    int32_t n_onchip_max;     /* largest on-chip subsystem for this device and dtype   */
    int32_t split_kp_max;     /* max levels per split pass                             */
    int32_t onchip_threads;   /* on-chip kernel CTA size                               */
    int32_t subsys_per_cta;   /* on-chip subsystems per CTA (1)                        */
    int32_t split_segments;   /* CTAs cooperating on one system in pass 1 (stage 1)    */
    int32_t split_tile_eff;   /* rows one split CTA produces per tile in pass 1        */
    int32_t chunks;           /* system chunks the batch is processed in               */
    int32_t launches;         /* kernel launches per solve (tds_solve_stages range)    */
    int64_t slot_rows;        /* workspace rows reserved per subsystem (final pass)    */
    size_t workspace_bytes;   /* bytes tds_solve_batched needs (0 when k == 0)         */
    int32_t onchip_form;      /* stage 3->4 form the on-chip kernel runs (16-byte aligned
                                 arrays): TDS_FORM_PCR_THOMAS = the paper's base kernel
                                 (PCR until T chains, Thomas per chain, §III-A) after c / c2
                                 CR levels; TDS_FORM_WARP_CR = CR in registers and across the
                                 32 lanes, shuffle PCR / CR on the per-warp top rows (T
                                 unused); -1 for a split-only plan                          */
} tds_plan_info;

enum { TDS_FORM_PCR_THOMAS = 0, TDS_FORM_WARP_CR = 1 };

/* ---- planning (host only, no device work) -------------------------------- */

/* Plan a solve of m systems of n equations on CUDA device `device` with the
 * DEFAULT or STATIC method.  *out receives a new plan (free with
 * tds_plan_destroy).  Errors: INVALID_ARG (n < 1, m < 1, 0 < batch_stride < n,
 * bad dtype/mode, out == NULL), CUDA (device query failed). */
tds_status tds_plan(tds_plan_t *out, int device, tds_dtype dtype, int64_t n, int64_t m,
                    int64_t batch_stride, tds_param_mode mode);

/* Same as tds_plan, from explicit (possibly fake) device properties (host
 * pointer, read only during the call).  The plan's device is -1: it can be
 * inspected but tds_solve_batched rejects it (DEVICE_MISMATCH). */
tds_status tds_plan_from_props(tds_plan_t *out, const tds_device_props *props, tds_dtype dtype,
                               int64_t n, int64_t m, int64_t batch_stride, tds_param_mode mode);

/* Fill *out (host) with the properties of CUDA device `device`. */
tds_status tds_device_props_query(int device, tds_device_props *out);

tds_status tds_plan_info_get(const tds_plan_t plan, tds_plan_info *out);

/* Replace the plan's tunable parameters (host struct) after validating them
 * against the kernels' limits; derived fields (n_sub, threads, workspace) are
 * recomputed and the plan's mode becomes TUNED.  INVALID_ARG / UNSUPPORTED on
 * a rejected set (the plan is then unchanged). */
tds_status tds_plan_set_params(tds_plan_t plan, const tds_params *params);

/* Canonical subsystem order after k levels (Fig. 3a): residue r
 * ascending, then row ascending: perm[off(r) + j] = r + 2^k j, off(r) =
 * sum_{r'<r} ceil((n - r')/2^k).  perm_host: host array of len == n entries. */
tds_status tds_plan_permutation(const tds_plan_t plan, int64_t *perm_host, int64_t len);

tds_status tds_plan_destroy(tds_plan_t plan);

/* ---- self-tuning (§IV-D) -------------------------------------- */

/* Tune the plan's switch points on its device: decoupled, seeded hill climb
 * over timed trials on generated diagonally dominant systems of the plan's
 * shape (the on-chip switch (c, T) and the split schedule (k, passes, tile,
 * theta) are searched independently, starting from the STATIC seed).
 * Allocates and frees its own device buffers; synchronises `cuda_stream`.
 * cache_path (host string, may be NULL => $TDS_TUNE_CACHE or no cache): a
 * text file of saved results keyed by device, dtype, n and m ("save those
 * results for future runs"); a hit skips the search.  A trial
 * is the median over several samples of back-to-back solves (>= ~0.4 ms per
 * sample; a solve under 30 us is timed as CUDA-graph replays of captured
 * solves on a private stream, since eager launches would time the host's
 * launch rate); the Thomas switch T is not searched in the warp form (no T);
 * the x placement (x_group) and the paper's load variant (strided 0 / 1 / 2)
 * are searched with the on-chip switch.  A
 * trial that faults the device (sticky CUDA error) aborts the search with
 * TUNE; the chosen parameters must reproduce the seed plan's x on the trial
 * systems (relative 2e-4 fp32 / 1e-9 fp64) before they and the cache line
 * are committed -- on any error the plan is unchanged.
 * Errors: INVALID_ARG, DEVICE_MISMATCH, NO_MEMORY, CUDA, TUNE. */
tds_status tds_tune(tds_plan_t plan, void *cuda_stream, const char *cache_path);

/* Trials run by the most recent tds_tune on this plan (0 on a cache hit). */
tds_status tds_plan_tune_trials(const tds_plan_t plan, int32_t *trials);

/* TEST-ONLY: tds_tune's search (§IV-D: decoupled stages, hill climb from the
 * plan's current parameters, 2 % ties, cache) with the trial cost supplied by
 * the caller instead of timed device solves -- no device work, so a plan from
 * tds_plan_from_props works.  cost (host callback): the "median time" of one
 * solve with *params (called only for parameter sets the planner accepts;
 * return >= 1e30 to refuse one, NaN to abort the search).  user is passed
 * through.  cache_path as in tds_tune.  tds_plan_tune_trials reports the
 * number of cost calls.  Errors: INVALID_ARG (NULL plan / cost), TUNE (the
 * seed was refused or the search aborted). */
tds_status tds_tune_search(tds_plan_t plan, double (*cost)(const tds_params *params, void *user), void *user,
                           const char *cache_path);

/* ---- solving ---------------------------------------------------------------- */

/* x = A^{-1} d for every system.  a, b, c, d: device, dtype, m x batch_stride.
 * x: device, same layout; may alias d exactly (in-place), must not otherwise
 * overlap a, b, c or d.  workspace: device, >= info.workspace_bytes bytes,
 * 256-byte aligned (may be NULL when info.workspace_bytes == 0); its contents
 * are scratch, undefined after the call (the kernels drop dead workspace lines
 * from L2 without writing them back).  Enqueued on cuda_stream; returns
 * immediately.  Errors (nothing enqueued): INVALID_ARG, WORKSPACE,
 * DEVICE_MISMATCH, UNSUPPORTED; CUDA on a launch failure. */
tds_status tds_solve_batched(const tds_plan_t plan, const void *a, const void *b, const void *c,
                             const void *d, void *x, void *workspace, size_t workspace_bytes,
                             void *cuda_stream);

/* Run only launches first_stage..last_stage (inclusive) of the kernel sequence
 * tds_solve_batched enqueues.  The sequence is, for each chunk of
 * chunk_systems systems in order: split passes 0..passes-1 (PAPER.md stages
 * 1-2), the on-chip kernel (stages 3-4) and, when k > 0, x_group == 0 and strided == 0, the x
 * placement; launch index = chunk * S + stage with
 * S = passes + 1 + (k > 0 && x_group == 0 && strided == 0), and
 * info.launches = chunks * S.  Calling every launch in order on one stream is
 * identical to tds_solve_batched (used to time each kernel with events between
 * them); each launch consumes what the previous one left in the workspace, so a
 * stage re-run without its predecessors reads undefined data.  Same arguments and errors as tds_solve_batched; INVALID_ARG if the
 * range is empty or outside [0, info.launches). */
tds_status tds_solve_stages(const tds_plan_t plan, const void *a, const void *b, const void *c,
                            const void *d, void *x, void *workspace, size_t workspace_bytes,
                            void *cuda_stream, int32_t first_stage, int32_t last_stage);

/* Diagnostic: run only the split stage (stages 1-2) and write the split
 * system in CANONICAL order, normalised so that b' = 1: for system s,
 * out[s*n + off(r) + j] holds the coefficient of original row r + 2^k j
 * (the tds_plan_permutation order).  a_out, c_out, d_out: device, dtype,
 * m x n (dense).  Requires k >= 1.  Same workspace rules as the solve. */
tds_status tds_split_batched(const tds_plan_t plan, const void *a, const void *b, const void *c,
                             const void *d, void *a_out, void *c_out, void *d_out,
                             void *workspace, size_t workspace_bytes, void *cuda_stream);

/* Same solve for NORMALISED systems (b = 1, the form every split pass leaves,
 * SURVEY.md §8(c)): a, c, d only, no b array is read.  a[0] and c[n-1] of
 * each system multiply identity rows and are ignored (they must be finite).
 * The plan needs k >= 1 and strided == 0 (the k = 0 on-chip kernels read b);
 * else UNSUPPORTED.  Otherwise as tds_solve_batched.  Used by the one-huge-
 * system path (dist.py solve_huge: the all-to-all delivers normalised residue
 * systems, so no b' = 1 array is materialised). */
tds_status tds_solve_normalized(const tds_plan_t plan, const void *a, const void *c, const void *d, void *x,
                                void *workspace, size_t workspace_bytes, void *cuda_stream);

/* Where the split passes leave the split system inside the workspace (host
 * only).  Three arrays a', c', d' of NORMALISED rows (b' = 1) start at element
 * offsets a_offset, c_offset, d_offset (elements of the plan's dtype from the
 * workspace base); slot (s << k) + r (r < 2^k, s < m) holds residue class r of
 * system s -- original rows r + 2^k j, j = 0 .. ceil((n - r) / 2^k) - 1 --
 * contiguously from element slot * slot_rows (Fig. 3a; canonical
 * order, R23).  UNSUPPORTED for k = 0, strided or chunked plans. */
typedef struct {
    int64_t a_offset, c_offset, d_offset;
    int64_t slot_rows;   /* elements between consecutive slots (>= ceil(n / 2^k)) */
    int64_t num_slots;   /* m * 2^k */
} tds_slots_layout;
tds_status tds_plan_slots_layout(const tds_plan_t plan, tds_slots_layout *out);

/* Run only the plan's split passes (PAPER.md stages 1-2), leaving the split
 * system in the workspace as tds_plan_slots_layout describes -- the zero-copy
 * source of the one-huge-system all-to-all (each residue class's rows of a
 * block are one contiguous run).  Split-only plans are accepted.  Same array,
 * workspace and device rules as tds_solve_batched; enqueued on cuda_stream. */
tds_status tds_split_slots(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                           void *workspace, size_t workspace_bytes, void *cuda_stream);

/* The split pass with the all-to-all of the one-huge-system path FUSED into
 * its output (the paper's Stage 1, over several GPUs): the plan's
 * ONE split pass (m = 1 system, k <= 8 levels, 16-byte aligned a, b, c, d)
 * writes residue class r = h q + rl (q = residues_per_group) straight into
 * destination h's arrays: normalised a', c', d' of position first_pos + j of
 * residue r go to dst[t][h][rl * dst_stride + j] for j in [0, num_pos) -- each
 * tile's outputs leave by TMA tensor stores, so on a multi-GPU node the
 * transfer to peer memory (dst pointers mapped from other GPUs, e.g. torch
 * symmetric memory over NVLink) overlaps the split tile by tile; positions
 * outside the window (the halo) are not written.  No workspace.  The caller
 * orders the destinations' readers after this call (a barrier across the
 * ranks).  first_pos, num_pos and dst_stride must be 16-byte multiples (TMA
 * tensor stores start -- and clip at the window's end -- on 16-byte
 * boundaries, measured on sm_100a; a store box starting before the window
 * -- the left halo -- leaves by plain stores: on sm_100a a TMA store with a
 * negative start coordinate is an illegal instruction).  Errors: INVALID_ARG
 * (NULL, groups not in [1, 8], groups * q != 2^k, window outside
 * floor(n / 2^k), dst_stride < num_pos, first_pos / num_pos / dst_stride not 16-byte
 * multiples, NULL / misaligned / overlapping dst), UNSUPPORTED (m != 1, not
 * one pass of <= 8 levels, misaligned inputs), CUDA. */
typedef struct {
    int32_t groups;             /* destinations (GPUs), <= 8                         */
    int32_t residues_per_group; /* q: residues [h q, (h+1) q) go to destination h    */
    int64_t first_pos;          /* first slot position stored of every residue       */
    int64_t num_pos;            /* positions stored per residue                      */
    int64_t dst_stride;         /* elements between consecutive residues at a dst    */
    void *dst[3][8];            /* [a', c', d'][destination]: device (or peer) bases */
} tds_scatter;
tds_status tds_split_scatter(const tds_plan_t plan, const void *a, const void *b, const void *c, const void *d,
                             const tds_scatter *spec, void *cuda_stream);

/* tds_solve_normalized with the x placement FUSED with the return of x to its
 * owners (the one-huge-system path's second all-to-all): rows
 * [h rows_per_group, (h+1) rows_per_group) of system s of x go to dst[h] +
 * s * dst_system_stride -- the placement kernel's TMA tensor stores write them
 * straight into (peer) memory.  Needs k >= 5, the TMA placement (n and
 * rows_per_group multiples of 2^k, rows_per_group / 2^k a multiple of
 * 4 * 128 / sizeof(T)), groups * rows_per_group == n, no chunking, strided 0,
 * x_group 0.  No x array; d is not written.  The caller orders the owners'
 * readers after the call (a barrier).  Errors: as tds_solve_normalized, plus
 * INVALID_ARG for the shape rules and NULL / misaligned / overlapping dst. */
typedef struct {
    int32_t groups;              /* destinations (GPUs), <= 8                 */
    int64_t rows_per_group;      /* rows of every system each destination owns */
    int64_t dst_system_stride;   /* elements between systems at a destination  */
    void *dst[8];                /* device (or peer) bases                     */
} tds_xscatter;
tds_status tds_solve_normalized_xscatter(const tds_plan_t plan, const void *a, const void *c, const void *d,
                                         const tds_xscatter *spec, void *workspace, size_t workspace_bytes,
                                         void *cuda_stream);

/* The residue-class -> original-order transpose of Fig. 3a:
 * x[s * batch_stride + r + 2^k j] = xs[((s << k) + r) * slot_rows + j] for
 * every system s < m, residue r < 2^k and row r + 2^k j < n.  xs, x: device,
 * dtype, must not overlap; xs is left intact.  The x placement kernel of the
 * solve (TMA transposer); also the unpacking of the one-huge-system x
 * return.  Errors: INVALID_ARG (k < 1, slot_rows < ceil(n/2^k), NULL,
 * misaligned, overlap), CUDA.  Enqueued on cuda_stream. */
tds_status tds_unpack_residues(tds_dtype dtype, int64_t n, int64_t m, int32_t k, int64_t slot_rows, const void *xs,
                               void *x, int64_t batch_stride, void *cuda_stream);

/* ---- batch-interleaved layout (ADI-style batches) ----- */

/* Bytes of device workspace tds_solve_interleaved needs for `plan`: the
 * plan's own workspace plus four system-major copies of the m x n arrays
 * (each rounded up to 256 bytes).  The plan must be dense (batch_stride == n).
 * Errors: INVALID_ARG (NULL), UNSUPPORTED (padded -- batch_stride != n -- or split-only plan). */
tds_status tds_interleaved_workspace_bytes(const tds_plan_t plan, size_t *bytes);

/* Same solve as tds_solve_batched for arrays in the INTERLEAVED layout:
 * element i of system s at ptr[i * m + s] (row-major n x m, the layout of
 * ADI sweeps along the fast axis).  The arrays are transposed into the
 * workspace by a shared-memory tile kernel (reads coalesced along systems,
 * writes along rows), solved by the plan's kernels in place, and x is
 * transposed back: 2 x 4 s extra HBM bytes per equation in, 2 s out.
 * x: device, interleaved, may alias d exactly.  workspace: device, 256-byte
 * aligned, >= tds_interleaved_workspace_bytes.  Same errors as
 * tds_solve_batched (plus UNSUPPORTED for a padded plan, batch_stride != n); enqueued on
 * cuda_stream, asynchronous. */
tds_status tds_solve_interleaved(const tds_plan_t plan, const void *a, const void *b, const void *c,
                                 const void *d, void *x, void *workspace, size_t workspace_bytes,
                                 void *cuda_stream);

/* ---- synthetic inputs ------------------------- */

/* Fill a, b, c, d (device, dtype, m x batch_stride; padding untouched) with the
 * seeded diagonally dominant systems of the input recipe, bit-identical to the
 * host generator (inputs.py, family "dd" with margin mu; "weak" is mu < 1):
 * h = splitmix64(seed ^ (array_id << 56) ^ ((first_system + s) * n + i)),
 * a, c, d = exact dyadic 2u - 1 from the top 24 (fp32) / 53 (fp64) bits of h
 * (array ids 0, 2, 3), a_0 = c_{n-1} = 0, b = (|a| + |c|) + mu rounded to
 * nearest in the target precision.  first_system: global index of system 0
 * (a rank of a sharded batch draws exactly the unsharded rows).  Enqueued on
 * cuda_stream.  Errors: INVALID_ARG (dtype, n < 1, m < 1, stride < n, NULL or
 * misaligned pointer), CUDA (launch). */
tds_status tds_generate(tds_dtype dtype, int64_t n, int64_t m, int64_t batch_stride, uint64_t seed,
                        int64_t first_system, double mu, void *a, void *b, void *c, void *d, void *cuda_stream);

/* Rows [row0, row0 + count) of ONE system of n rows drawn by the same recipe
 * (global_row = row; a_0 = c_{n-1} = 0), rows outside [0, n) as identity rows
 * (a, b, c, d) = (0, 1, 0, 0): the halo-padded row block a rank of the
 * one-huge-system path owns.  a, b, c, d: device, count elements each.
 * Errors as tds_generate. */
tds_status tds_generate_rows(tds_dtype dtype, int64_t n, int64_t row0, int64_t count, uint64_t seed, double mu,
                             void *a, void *b, void *c, void *d, void *cuda_stream);

/* ---- misc ---------------------------------------------------------------------- */

const char *tds_status_string(tds_status status);
const char *tds_last_error(void);
int tds_version(void);

#ifdef __cplusplus
}
#endif
#endif /* TDS_H_ */

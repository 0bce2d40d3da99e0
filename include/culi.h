/* =====================================================================================================
 * culi.h — C-ABI of libculi.so, the B200-native (sm_100a) hot path of CuLi
 * ("And Now for Something Completely Different: Running Lisp on GPUs", Süß, Döring, Brinkmann, Nagel;
 * /root/reference/PAPER.md, cited "PAPER Lnnn §x").
 *
 * The calls follow the paper's read-eval-print split: the host reads text into a compact node array
 * (§III-B.b, moved to the host per L85-89), `culi_define` persists global bindings on the
 * device (the global environment persists for the session, L98-101, L389), `culi_eval_batch` evaluates N
 * independent forms on the device (eval: L438-462 §III-B.c; independent parallel evaluation: L546-589
 * §III-D), and results are copied back for printing on the host (L463-475 §III-B.d).
 * Semantics of every form are SURVEY.md §8(c) / DESIGN.md §3.
 *
 * Conventions (all entry points):
 *   - Return value: 0 = CULI_OK, negative = API failure (culi_status).  Lisp-level errors (type errors,
 *     arity, depth, fuel ...) are NOT API failures: they are per-form result codes (culi_err).
 *   - Plain pointers and sizes only.  Host pointers unless the name says dev_*.
 *   - Ownership: the caller owns every buffer it passes in (text, out buffers, device buffers given in
 *     culi_opts).  The library owns culi_ctx / culi_image / culi_results until the matching *_free /
 *     culi_shutdown.  No call retains a caller pointer after it returns, except opts->stream.
 *   - Threading: one ctx per host thread; every device operation of a ctx is ordered on opts->stream.
 *   - There is no CPU fallback: without a usable CUDA device culi_init fails with CULI_E_CUDA.
 * ===================================================================================================== */
#ifndef CULI_H
#define CULI_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef enum {
  CULI_OK = 0,
  CULI_E_ARG = -1,        /* bad argument, NULL pointer, buffer too small (needed size reported)      */
  CULI_E_PARSE = -2,      /* read error: unbalanced parens (L484-486), unterminated string, int64
                             literal out of range; *err_offset = byte offset                             */
  CULI_E_HEAP_FULL = -3,  /* device heap / stacks exhausted: the batch results are invalid            */
  CULI_E_CUDA = -4,       /* a CUDA runtime call failed (no device, launch failure ...)               */
  CULI_E_NCCL = -5,       /* reserved for collective failures reported by the caller's binding          */
  CULI_E_DEFINE = -6,     /* culi_define: a definition form evaluated to an error (*failed_index)       */
  CULI_E_STATE = -7       /* call out of order (e.g. import into a ctx that already has definitions)   */
} culi_status;

/* Per-form Lisp error codes.  CULI_ERR_OOM is a resource error, never parity-checked. */
typedef enum {
  CULI_ERR_NONE = 0, CULI_ERR_TYPE = 1, CULI_ERR_ARITY = 2, CULI_ERR_DIV0 = 3, CULI_ERR_SYNTAX = 4,
  CULI_ERR_ARG = 5, CULI_ERR_DEPTH = 6, CULI_ERR_FUEL = 7, CULI_ERR_DEFINE_IN_BATCH = 8, CULI_ERR_OOM = 9
} culi_err;

/* Value tags as reported by culi_result_info. */
typedef enum {
  CULI_NIL = 0, CULI_T = 1, CULI_INT = 2, CULI_FLOAT = 3, CULI_STRING = 4, CULI_SYMBOL = 5,
  CULI_CONS = 6, CULI_BUILTIN = 7, CULI_SPECIAL = 8, CULI_CLOSURE = 9, CULI_MACRO = 10,
  CULI_ERROR = 13
} culi_tag;

typedef struct culi_ctx culi_ctx;
typedef struct culi_image culi_image;
typedef struct culi_results culi_results;

typedef struct {
  int device;              /* CUDA device ordinal                                                       */
  void* stream;            /* cudaStream_t (e.g. torch.cuda.current_stream().cuda_stream); NULL = the
                              legacy default stream.  Borrowed: must outlive the ctx.                    */
  uint64_t heap_nodes;     /* node capacity of the heap (16-byte nodes: word u64 + tag u8, loaded with one
                              16-byte access); 0 = default (64 Mi nodes = 1 GiB).  The paper's node array was fixed at compile time
                              (L361-365); here it is sized at init.                                     */
  uint32_t max_depth;      /* canonical eval-nesting limit (c.10); 0 = default 1024; at most 4095         */
  uint64_t fuel;           /* canonical step limit per top-level form (c.10); 0 = default 2^40            */
  uint32_t vstack_entries; /* value-stack entries per resident thread; 0 = default 4096                   */
  uint32_t slots;          /* resident eval threads (stack slots); 0 = default (SM count x 1024)         */
  uint32_t flags;          /* CULI_F_* below                                                              */
  void* heap_base;         /* caller-owned device memory for the heap, global table, string area and
                              stacks (e.g. a torch uint8 tensor's data_ptr); NULL = the library
                              cudaMallocs them.  Borrowed: must outlive the ctx; 256-byte aligned.        */
  uint64_t heap_bytes;     /* size of heap_base; at least culi_arena_bytes(opts) (CULI_E_ARG otherwise)   */
} culi_opts;

/* Bytes of device memory a ctx with these opts places in heap_base (the heap's node array, the global
 * frame, the string area, K- and V-stacks; SURVEY §8(d) "heap and stack budget").  The remaining session
 * state (counters, descriptors, result buffers) stays library-allocated. */
int culi_arena_bytes(const culi_opts* opts, uint64_t* bytes);

#define CULI_F_NO_BINNING 1u   /* evaluate forms in input order (no classify+sort dispatch, §8(a)5)     */
#define CULI_F_NO_FANOUT  2u   /* evaluate top-level ||| forms in one thread (no fan-out, §8(a)6)        */
#define CULI_F_NO_STAGING 4u   /* do not stage the global frame / hot code in shared memory (§8(a)4)     */
#define CULI_F_NO_VOTING  8u   /* batches that neither split nor nest: plain kernel instead of the warp-voting
                                  one (lanes regroup by stack height + continuation at returns) */
#define CULI_F_NO_NESTED 16u   /* run nested (non-top-level) ||| forms and wide data lists / (list ...)
                                  below the top level inside one thread (§8(f)1 off)      */
#define CULI_F_NO_SPLIT  32u   /* no argument splitting: each form is evaluated by one thread only        */
#define CULI_F_NO_GC     64u   /* do not compact the persistent heap segment after culi_define (§8(f)3)  */
#define CULI_F_NO_GRAPH 128u   /* culi_eval_uploaded issues its launches directly (no CUDA-graph replay)  */
#define CULI_F_DEVICE_READ 256u /* culi_eval_text / culi_upload_text: always read on the device.  Without it
                                  (and without env CULI_DEVICE_READ=1) host text of at most 16 KiB is read
                                  by the host reader (same image): below that size the device
                                  reader's launches and 3 sync points cost more than the parse itself      */
/* Without flags: batches of <= 4,096 forms with no lambda / defun in them or in any definition run in
 * input order (no dispatch) and without argument splitting; argument splitting runs wherever a closure can
 * exist (binned or not, CULI_F_NO_BINNING included) — DESIGN.md §5.5. */

/* Fill *opts with defaults (device 0, default stream, default sizes). */
void culi_default_opts(culi_opts* opts);

/* Create a session: allocates the device heap, stacks and global table on opts->device and installs the
 * builtins and special forms in the global environment (the master thread set up the
 * global environment; here it is one host->device copy).  Returns CULI_E_CUDA without a device. */
int culi_init(const culi_opts* opts, culi_ctx** out);
void culi_shutdown(culi_ctx* ctx);

/* ---- read (host) ---------------------------------------------------------------------------------
 * Parse `len` bytes of text into a compact node image; every top-level
 * datum is one form.  Symbols are interned into ctx's table (dense u32 ids).  On CULI_E_PARSE,
 * *err_offset (if non-NULL) receives the byte offset of the offending character / opening paren. */
int culi_read(culi_ctx* ctx, const char* text, size_t len, culi_image** out, size_t* err_offset);
uint32_t culi_image_nforms(const culi_image* img);
/* Page-lock the image's host arrays (cudaHostRegister) so that uploads DMA them from pinned memory.
 * Idempotent; undone by culi_image_free.  *h2d_bytes (if non-NULL) = bytes an upload of it copies. */
int culi_image_pin(culi_image* img, uint64_t* h2d_bytes);
uint64_t culi_image_nnodes(const culi_image* img);
void culi_image_free(culi_image* img);

/* ---- define (device, sequential) -----------------------------------------------------------------
 * Upload `defs` into the persistent heap segment and evaluate its forms in order on the device with
 * define/defun/defmacro enabled; bindings persist until culi_shutdown (L98-101, L316-319, L346-347).
 * Stops at the first form whose evaluation errors: returns CULI_E_DEFINE, *failed_index = its index,
 * *failed_err = its culi_err; that binding is not created (earlier ones stay). */
int culi_define(culi_ctx* ctx, const culi_image* defs, uint32_t* failed_index, uint8_t* failed_err);
/* (culi_define / culi_define_text while a batch is uploaded with culi_upload*: CULI_E_STATE — the new
 * definitions would land below the uploaded batch; culi_release it first.) */

/* ---- eval (device, data-parallel) ------------------------------------------------------------------
 * Evaluate the image's forms as N independent evaluations (one thread each; top-level ||| forms fan out
 * over threads).  The global environment is read-only: define/defun/defmacro yield the
 * per-form error CULI_ERR_DEFINE_IN_BATCH.  Synchronous on ctx's stream: on return the results (records
 * + serialized list/string values) are in host memory and the batch's heap segment has been released.
 * On CULI_E_HEAP_FULL no results are returned. */
int culi_eval_batch(culi_ctx* ctx, const culi_image* forms, culi_results** out);

/* Asynchronous variant (the paper's host-reads / device-evaluates split, L85-89, L477-480): uploads the
 * image and enqueues dispatch + eval + export on ctx's stream, then returns without waiting; *out is a
 * results object that is NOT ready (every accessor returns CULI_E_STATE) until culi_sync(ctx) completes
 * it (D2H of records + payload; sequential fallbacks run there).  The host may read the next batch
 * meanwhile.  One batch in flight per ctx: a second call before culi_sync returns CULI_E_STATE.  The image
 * must stay alive until culi_sync (pin it with culi_image_pin for a true async H2D). */
int culi_eval_batch_async(culi_ctx* ctx, const culi_image* forms, culi_results** out);
/* Wait for the batch started by culi_eval_batch_async and complete its results (no-op without one). */
int culi_sync(culi_ctx* ctx);

/* Device-resident variant for timing (bench.py "value"): the image must already be uploaded with
 * culi_upload (done once); each call runs relocate-free dispatch + eval + export on the device and
 * leaves records on the device.  No host copies, no host synchronisation.  On a non-default stream the
 * first call captures the step into a CUDA graph and later calls replay it (CULI_F_NO_GRAPH: no graph). */
int culi_upload(culi_ctx* ctx, const culi_image* forms, uint32_t* batch_handle);
int culi_eval_uploaded(culi_ctx* ctx, uint32_t batch_handle);
/* Complete the device-resident results of the last culi_eval_uploaded call without copying them to the
 * host: sequential re-evaluation of undecided ||| forms, eval + export again into a grown payload buffer
 * (synchronises).  Used before culi_results_export on the end-to-end multi-GPU path. */
int culi_complete(culi_ctx* ctx, uint32_t batch_handle);
/* Copy the device-resident results of the last culi_eval_uploaded call to the host (synchronises). */
int culi_fetch_results(culi_ctx* ctx, uint32_t batch_handle, culi_results** out);
/* Release an uploaded batch (resets the heap to the post-define mark). */
int culi_release(culi_ctx* ctx, uint32_t batch_handle);

/* ---- device reader -----------------------------------------------------------------
 * The paper reads on the GPU (§III-B.b) and found parsing to be the dominant GPU
 * phase (L785-788, L1081-1088); these calls read program text ON THE DEVICE, straight into the heap: a
 * data-parallel lexer (scan of per-byte transition functions), a bracket-depth scan, token
 * classification + int64 / correctly rounded binary64 parsing, device symbol interning (same dense ids as
 * culi_read, so printing and the global environment are shared), a stable (depth, item) radix sort that
 * groups list elements, and node emission with contiguous spines (c.14).  The image and every result are
 * identical to culi_read + culi_define / culi_eval_batch on the same text (syntax: SURVEY §8(c).1).
 *   text, len      : `len` bytes of program text (len < 2^32 - 1).  text_on_device != 0: a device pointer
 *                    (any alignment; 16-byte aligned reads when aligned), else host memory (copied to the
 *                    device first; page-locked memory copies fastest).  Borrowed for the call only.
 *   err_offset     : on CULI_E_PARSE, the same byte offset culi_read reports (first offending character,
 *                    else the innermost construct still open at the end of the text).
 * culi_define_text: culi_define on the read forms (same failure reporting).
 * culi_eval_text  : culi_eval_batch on the read forms (synchronous, results on the host).
 * culi_upload_text: read + prepare a batch for culi_eval_uploaded / culi_fetch_results (*nforms = forms).
 * culi_last_read  : device time in ms of the last device read (lex .. emit, text already in HBM), its
 *                   item count (structural characters + datum starts) and the nodes it emitted. */
int culi_define_text(culi_ctx* ctx, const char* text, size_t len, int text_on_device, uint32_t* failed_index,
                     uint8_t* failed_err, size_t* err_offset);
int culi_eval_text(culi_ctx* ctx, const char* text, size_t len, int text_on_device, culi_results** out,
                   size_t* err_offset);
int culi_upload_text(culi_ctx* ctx, const char* text, size_t len, int text_on_device, uint32_t* batch_handle,
                     uint32_t* nforms, size_t* err_offset);
int culi_last_read(const culi_ctx* ctx, float* ms, uint64_t* items, uint64_t* nodes);

/* ---- heap reclamation ----------------------------------------------------------------
 * The paper hands out "the sequentially next free node" of a fixed node array and marks nodes that are no
 * longer needed as free (§III-A.c).  Batch allocations are released wholesale after every
 * batch; the persistent segment (definitions and what their evaluation allocated) is compacted on the
 * device after every culi_define / culi_define_text unless CULI_F_NO_GC: nodes reachable from the global
 * environment are kept (mark from the global table, contiguous cons runs traced as one object) and slid
 * down in address order, so contiguous list spines stay contiguous (c.14) and results are unchanged.
 * culi_collect   : run the compaction now (not while a batch is uploaded: CULI_E_STATE).  *live_nodes =
 *                  nodes kept, *freed_nodes = nodes reclaimed.  Without scratch room above the segment
 *                  (2 x live > capacity) the segment is left as it is (freed = 0).
 * culi_heap_usage: *persistent_nodes = heap nodes in use between batches (the post-define mark, including
 *                  nodes 0/1), *capacity = heap nodes, *freed_total = nodes reclaimed so far. */
int culi_collect(culi_ctx* ctx, uint64_t* live_nodes, uint64_t* freed_nodes);
int culi_heap_usage(const culi_ctx* ctx, uint64_t* persistent_nodes, uint64_t* capacity, uint64_t* freed_total);

/* ---- results (host) --------------------------------------------------------------------------------- */
uint32_t culi_results_count(const culi_results* r);
/* tag: culi_tag (CULI_ERROR when err != 0); err: culi_err; steps: canonical eval steps (c.4). */
int culi_result_info(const culi_results* r, uint32_t i, uint8_t* tag, uint8_t* err, uint64_t* steps);
int culi_result_int(const culi_results* r, uint32_t i, int64_t* v);     /* CULI_E_ARG if not INT      */
int culi_result_float(const culi_results* r, uint32_t i, double* v);    /* CULI_E_ARG if not FLOAT    */
/* Print result i into buf[cap] (NUL-terminated).  *needed = length without the NUL,
 * always set; if cap <= *needed the text is truncated and CULI_E_ARG is returned. */
int culi_print(const culi_results* r, uint32_t i, char* buf, size_t cap, size_t* needed);
/* Sum of steps over all forms, and the number of forms with err != 0. */
int culi_results_totals(const culi_results* r, uint64_t* total_steps, uint32_t* n_errors);
void culi_results_free(culi_results* r);
/* Bytes the fetch of these results copied device -> host (records + serialized value tokens). */
int culi_results_wire_bytes(const culi_results* r, uint64_t* d2h_bytes);

/* ---- distributed hooks ------------------------------------------------------------------
 * The collective itself is issued by the caller (torch.distributed NCCL broadcast / all_gather) on a
 * device buffer, ordered on ctx's stream.
 * culi_env_export: pack the global environment (global table + persistent heap segment + symbol names)
 *   into dev_buf[cap] (device memory).  *bytes = size needed (always set); CULI_E_ARG if cap too small.
 * culi_env_import: replace this ctx's (empty) global environment by the packed image in dev_buf; the
 *   ctx must not have run culi_define yet (CULI_E_STATE otherwise).  Both synchronise ctx's stream. */
int culi_env_export(culi_ctx* ctx, void* dev_buf, size_t cap, size_t* bytes);
int culi_env_import(culi_ctx* ctx, const void* dev_buf, size_t bytes);
/* Serialize host results into a self-contained byte blob (records + payload + symbol names) and
 * rebuild results from per-rank blobs: form_index[rank][k] = global index of that rank's k-th form. */
/* Pack the device-resident records of the last culi_eval_uploaded call into dev_buf (device memory, for
 * an NCCL all_gather): [tag u8 x n][err u8 x n][pad to 8][steps u64 x n][word u64 x n].  Stream-ordered,
 * no host synchronisation.  *bytes = size needed (always set); CULI_E_ARG if cap is too small. */
int culi_records_device(culi_ctx* ctx, void* dev_buf, size_t cap, size_t* bytes);
/* Device-resident result gather (the multi-GPU form of the paper's ordered result assembly,
 * PAPER L584-589).  culi_results_export packs the results of the ctx's current batch (after
 * culi_eval_uploaded; before culi_release) into dev_buf (device memory, for an NCCL all_gather of
 * fixed-size buffers): a 64-byte header {magic "CULIRES2", nforms, npayload, names_bytes, nstr, payload
 * capacity, overflow, 0}, then tag u8[n], err u8[n], steps u64[n], word u64[n] (8-aligned), the symbol
 * names (NUL-separated, id order) and string bytes, then the payload tokens (16 B each, 16-aligned).
 * Stream-ordered and without a host synchronisation: the token count is read on the device; tokens beyond
 * the capacity left in dev_buf are dropped and the header's overflow flag is set.  With dev_buf == NULL,
 * *bytes = the exact size these results need (this synchronises); otherwise *bytes = the fixed part +
 * the payload capacity used.  CULI_E_ARG if cap cannot hold the fixed part. */
int culi_results_export(culi_ctx* ctx, void* dev_buf, size_t cap, size_t* bytes);
/* Merge per-rank exported buffers (device pointers, e.g. slices of the all_gather output on this ctx's
 * device) into one host result set: records are scattered by global form index on the device, payload
 * tokens concatenated with their offsets shifted, SYMBOL tokens re-interned by name, STRING offsets
 * shifted; then one D2H.  form_index[r][k] = global index of rank r's k-th form, or form_index == NULL for
 * the strided deal of SURVEY §8(e) (rank r's k-th form is r + k * nranks).  CULI_E_ARG on a bad buffer or
 * an overflowed export (re-export with a larger capacity). */
int culi_results_import(culi_ctx* ctx, const void* const* dev_bufs, const size_t* sizes, int nranks,
                        const uint32_t* const* form_index, culi_results** merged);
int culi_results_serialize(const culi_results* r, void* buf, size_t cap, size_t* bytes);
int culi_results_merge(const void* const* blobs, const size_t* sizes, int nranks,
                       const uint32_t* const* form_index, culi_results** merged);

/* ---- diagnostics ---------------------------------------------------------------------------------- */
const char* culi_status_string(int status);
const char* culi_error_name(uint8_t err);
/* Device time in ms of the phases of the last eval call: [0] dispatch, [1] eval, [2] export; and the
 * number of kernels launched by that call.  Heap high-water mark in nodes. */
int culi_last_timing(const culi_ctx* ctx, float* ms3, uint32_t* kernels, uint64_t* heap_high);
/* Path statistics of the last fetched batch: forms handled by the fan-out kernels (top-level ||| forms
 * and wide forms), nested ||| evaluations that suspended and fanned out (§8(f)1),
 * and forms re-evaluated sequentially (an element error, fuel overflow, a short / non-contiguous list). */
int culi_last_stats(const culi_ctx* ctx, uint32_t* fanout_forms, uint32_t* fallback_forms,
                    uint32_t* nested_forms);
/* Argument splitting (an implementation choice, not a paper mechanism): the number of
 * split groups the last fetched batch published — each group is the pending arguments of the lanes of one
 * warp that polled together while an idle warp waited for work; the idle warp evaluates the group (or the
 * owners take it back).  Results, steps and errors are identical with CULI_F_NO_SPLIT.  0 for batches that
 * do not split (see the note after the CULI_F_* flags). */
int culi_last_splits(const culi_ctx* ctx, uint32_t* groups);
/* Of those, the groups an idle warp claimed and evaluated (the others were taken back by their owners). */
int culi_last_split_claims(const culi_ctx* ctx, uint32_t* claimed);
/* Every wait of one lane on another (an owner joining a split argument, a thief waiting for its group, a
 * nested ||| waiting for its elements) is bounded by 10 s (env CULI_WAIT_MS).  A wait that gives up
 * recovers exactly — the owner evaluates the argument itself / the form goes to the sequential fallback —
 * so results are unaffected; it is counted here for the last fetched batch (*timeouts; 0 in a healthy
 * run), and diag9 (if non-NULL, 9 entries) receives the first one's state: kind (1 join, 2 queue entry,
 * 3 nested), group (or descriptor), lane, form, group state, task mask, owners remaining, task done
 * flag, thief warp. */
int culi_last_waits(const culi_ctx* ctx, uint32_t* timeouts, uint32_t* diag9);
/* Work the last fetch (culi_fetch_results / culi_eval_batch / culi_eval_text) did after the device step it
 * fetched: forms re-evaluated by the sequential fallback (as culi_last_stats), and re-runs of eval + export
 * because the result payload buffer had to grow.  A timed culi_eval_uploaded step does neither; a caller
 * timing only that step checks both are 0 (bench.py does). */
int culi_last_reruns(const culi_ctx* ctx, uint32_t* fallback_forms, uint32_t* payload_regrows);

#ifdef __cplusplus
}
#endif
#endif /* CULI_H */

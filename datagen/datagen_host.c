/*
 * datagen_host.c — host (CPU) fill routines over ocl_datagen.h.
 * Input generation only: no method arithmetic lives here (see ocl_datagen.h).
 * Built with gcc -pthread into datagen/liboclgen_host.so.
 */
#include <math.h>
#include <pthread.h>
#include <stddef.h>
#include <stdint.h>
#include <unistd.h>
#include "ocl_datagen.h"

/* Minimal pthread parallel-for over [0, n) in contiguous chunks. */
typedef void (*oclg_body)(void* ctx, int64_t begin, int64_t end);
typedef struct { oclg_body fn; void* ctx; int64_t begin, end; } oclg_task;
static void* oclg_run(void* p) { oclg_task* t = (oclg_task*)p; t->fn(t->ctx, t->begin, t->end); return NULL; }
static void oclg_parallel_for(int64_t n, oclg_body fn, void* ctx) {
  long nt = sysconf(_SC_NPROCESSORS_ONLN);
  if (nt < 1) nt = 1;
  if (nt > 64) nt = 64;
  if (n < 65536) nt = 1;
  pthread_t th[64];
  oclg_task tasks[64];
  for (long t = 0; t < nt; ++t) {
    tasks[t].fn = fn; tasks[t].ctx = ctx;
    tasks[t].begin = n * t / nt; tasks[t].end = n * (t + 1) / nt;
    if (nt == 1) { oclg_run(&tasks[t]); return; }
    pthread_create(&th[t], NULL, oclg_run, &tasks[t]);
  }
  for (long t = 0; t < nt; ++t) pthread_join(th[t], NULL);
}

/* Fill rows [row0, row0+n) of the lineitem-shaped table.  Any output pointer may
 * be NULL.  f64 outputs hold the scale-2 decimal divided by 100.0.
 * If shuffled != 0, output row i is lineitem row feistel(i) of a table of
 * n_total rows (config C3 "shuffled" layout). */
typedef struct {
  uint64_t seed, row0, n_total; int shuffled;
  int64_t* orderkey; int32_t* shipdate; uint8_t* returnflag; uint8_t* linestatus;
  int64_t *quantity, *extendedprice, *discount, *tax;
  double *quantity_f, *extendedprice_f, *discount_f, *tax_f;
} li_ctx;

static void li_body(void* p, int64_t begin, int64_t end) {
  li_ctx* c = (li_ctx*)p;
  uint64_t seed = c->seed, row0 = c->row0, n_total = c->n_total;
  int shuffled = c->shuffled;
  int64_t* orderkey = c->orderkey; int32_t* shipdate = c->shipdate;
  uint8_t* returnflag = c->returnflag; uint8_t* linestatus = c->linestatus;
  int64_t *quantity = c->quantity, *extendedprice = c->extendedprice, *discount = c->discount, *tax = c->tax;
  double *quantity_f = c->quantity_f, *extendedprice_f = c->extendedprice_f, *discount_f = c->discount_f, *tax_f = c->tax_f;
  uint64_t nparts = oclg_nparts_for_rows(n_total);
  for (int64_t i = begin; i < end; ++i) {
    uint64_t r = row0 + (uint64_t)i;
    if (shuffled) r = oclg_feistel(seed, n_total, r);
    oclg_lineitem_row x = oclg_lineitem(seed, r, nparts);
    if (orderkey) orderkey[i] = x.orderkey;
    if (shipdate) shipdate[i] = x.shipdate;
    if (returnflag) returnflag[i] = x.returnflag;
    if (linestatus) linestatus[i] = x.linestatus;
    if (quantity) quantity[i] = x.quantity;
    if (extendedprice) extendedprice[i] = x.extendedprice;
    if (discount) discount[i] = x.discount;
    if (tax) tax[i] = x.tax;
    if (quantity_f) quantity_f[i] = (double)x.quantity / 100.0;
    if (extendedprice_f) extendedprice_f[i] = (double)x.extendedprice / 100.0;
    if (discount_f) discount_f[i] = (double)x.discount / 100.0;
    if (tax_f) tax_f[i] = (double)x.tax / 100.0;
  }
}

void oclg_fill_lineitem(uint64_t seed, uint64_t row0, uint64_t n, uint64_t n_total, int shuffled,
                        int64_t* orderkey, int32_t* shipdate, uint8_t* returnflag, uint8_t* linestatus,
                        int64_t* quantity, int64_t* extendedprice, int64_t* discount, int64_t* tax,
                        double* quantity_f, double* extendedprice_f, double* discount_f, double* tax_f) {
  li_ctx c = {seed, row0, n_total, shuffled, orderkey, shipdate, returnflag, linestatus, quantity, extendedprice,
              discount, tax, quantity_f, extendedprice_f, discount_f, tax_f};
  oclg_parallel_for((int64_t)n, li_body, &c);
}

/* Zipf(s) inverse-CDF table over G ranks: cdf[i] = sum_{k<=i} k^-s / H. */
void oclg_zipf_cdf(uint64_t G, double s, double* cdf) {
  double h = 0.0;
  for (uint64_t i = 0; i < G; ++i) h += pow((double)(i + 1), -s);
  double acc = 0.0;
  for (uint64_t i = 0; i < G; ++i) {
    acc += pow((double)(i + 1), -s);
    cdf[i] = acc / h;
  }
  cdf[G - 1] = 1.0;
}

typedef struct { uint64_t seed, row0, G; const double* cdf; int32_t* p; int64_t* key; int64_t* v; double* v_f; } sw_ctx;

static void sw_body(void* pc, int64_t begin, int64_t end) {
  sw_ctx* c = (sw_ctx*)pc;
  uint64_t seed = c->seed, row0 = c->row0, G = c->G;
  const double* cdf = c->cdf;
  int32_t* p = c->p; int64_t* key = c->key; int64_t* v = c->v; double* v_f = c->v_f;
  for (int64_t i = begin; i < end; ++i) {
    uint64_t r = row0 + (uint64_t)i;
    if (p) p[i] = oclg_sweep_p(seed, r);
    if (key) key[i] = oclg_sweep_key(seed, oclg_sweep_rank(seed, r, G, cdf));
    int64_t vv = oclg_sweep_v(seed, r);
    if (v) v[i] = vv;
    if (v_f) v_f[i] = (double)vv / 100.0;
  }
}

void oclg_fill_sweep(uint64_t seed, uint64_t row0, uint64_t n, uint64_t G, const double* cdf,
                     int32_t* p, int64_t* key, int64_t* v, double* v_f) {
  sw_ctx c = {seed, row0, G, cdf, p, key, v, v_f};
  oclg_parallel_for((int64_t)n, sw_body, &c);
}

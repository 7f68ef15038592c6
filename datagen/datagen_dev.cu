// datagen_dev.cu — device (sm_100a) fill kernels over ocl_datagen.h, so a GPU
// rank generates its row shard in place (SURVEY.md §8(d) "Generator").
// Input generation only: no method arithmetic lives here.  Built into
// datagen/liboclgen_dev.so; exported with a plain C ABI (device pointers).
#include <cuda_runtime.h>
#include <stdint.h>
#include "ocl_datagen.h"

namespace {

__global__ void k_fill_lineitem(uint64_t seed, uint64_t row0, uint64_t n, uint64_t n_total, int shuffled,
                                int64_t* orderkey, int32_t* shipdate, uint8_t* returnflag, uint8_t* linestatus,
                                int64_t* quantity, int64_t* extendedprice, int64_t* discount, int64_t* tax,
                                double* quantity_f, double* extendedprice_f, double* discount_f, double* tax_f) {
  uint64_t nparts = oclg_nparts_for_rows(n_total);
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t r = row0 + i;
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
    if (quantity_f) quantity_f[i] = __ddiv_rn((double)x.quantity, 100.0);
    if (extendedprice_f) extendedprice_f[i] = __ddiv_rn((double)x.extendedprice, 100.0);
    if (discount_f) discount_f[i] = __ddiv_rn((double)x.discount, 100.0);
    if (tax_f) tax_f[i] = __ddiv_rn((double)x.tax, 100.0);
  }
}

__global__ void k_fill_sweep(uint64_t seed, uint64_t row0, uint64_t n, uint64_t G, const double* cdf,
                             int32_t* p, int64_t* key, int64_t* v, double* v_f) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t r = row0 + i;
    if (p) p[i] = oclg_sweep_p(seed, r);
    if (key) key[i] = oclg_sweep_key(seed, oclg_sweep_rank(seed, r, G, cdf));
    int64_t vv = oclg_sweep_v(seed, r);
    if (v) v[i] = vv;
    if (v_f) v_f[i] = __ddiv_rn((double)vv, 100.0);
  }
}

int grid_for(uint64_t n) {
  int dev = 0, sms = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
  uint64_t blocks = (n + 255) / 256;
  uint64_t cap = (uint64_t)sms * 8;
  return (int)(blocks < cap ? (blocks ? blocks : 1) : cap);
}

}  // namespace

extern "C" int oclg_dev_fill_lineitem(uint64_t seed, uint64_t row0, uint64_t n, uint64_t n_total, int shuffled,
                                      int64_t* orderkey, int32_t* shipdate, uint8_t* returnflag, uint8_t* linestatus,
                                      int64_t* quantity, int64_t* extendedprice, int64_t* discount, int64_t* tax,
                                      double* quantity_f, double* extendedprice_f, double* discount_f, double* tax_f,
                                      void* stream) {
  if (n == 0) return 0;
  k_fill_lineitem<<<grid_for(n), 256, 0, (cudaStream_t)stream>>>(seed, row0, n, n_total, shuffled, orderkey, shipdate,
                                                                   returnflag, linestatus, quantity, extendedprice,
                                                                   discount, tax, quantity_f, extendedprice_f,
                                                                   discount_f, tax_f);
  return (int)cudaGetLastError();
}

extern "C" int oclg_dev_fill_sweep(uint64_t seed, uint64_t row0, uint64_t n, uint64_t G, const double* cdf_dev,
                                   int32_t* p, int64_t* key, int64_t* v, double* v_f, void* stream) {
  if (n == 0) return 0;
  k_fill_sweep<<<grid_for(n), 256, 0, (cudaStream_t)stream>>>(seed, row0, n, G, cdf_dev, p, key, v, v_f);
  return (int)cudaGetLastError();
}

// Un-permute of the cyclic-row Mandelbrot image (mandelbrot_cyclic.cu): an
// index Map over the row-major pixel pairs that reads each pair from its slot
// of the permuted image (a vector argument holding the whole permuted image:
// single or copy distribution).  Row r sits in slot (r mod D)*R + r div D.
struct Cnt2 { int n0, n1; };
Cnt2 mandelbrot_unpermute(unsigned i, const Cnt2 *perm, int width, int height, int D) {
    const unsigned half = (unsigned)width / 2u;
    const unsigned row = i / half, pc = i % half;
    const unsigned R = ((unsigned)height + (unsigned)D - 1u) / (unsigned)D;
    const unsigned slot = (row % (unsigned)D) * R + row / (unsigned)D;
    return perm[(unsigned long long)slot * half + pc];
}

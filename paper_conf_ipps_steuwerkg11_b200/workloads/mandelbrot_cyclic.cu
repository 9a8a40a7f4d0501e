
// ---- cyclic rows, appended to mandelbrot_pairs.cu ----
// The paper distributes the image's rows in blocks, so
// the device holding the middle rows (most of the set) does most of the work:
// at 8 devices the busiest has 3.1x the mean.  Here an index Map over a
// PERMUTED row order gives device k the rows k, k+D, k+2D, ...: with the
// output block-distributed, slot s of the permuted image (s = k*R + t,
// R = ceil(H/D) slots per device) holds row k + t*D.  Pixels go two per
// element (mandelbrot_pairs); slots past the last row are padding (0, 0).
// mandelbrot_unpermute.cu puts the rows back in row-major order.
// c is computed exactly as the position vector of the plain Map (reading R5).
Cnt2 mandelbrot_cyclic(unsigned j, int width, int height, int cap, int D) {
    const unsigned half = (unsigned)width / 2u;
    const unsigned slot = j / half, pc = j % half;
    const unsigned R = ((unsigned)height + (unsigned)D - 1u) / (unsigned)D;
    const unsigned row = slot / R + (slot % R) * (unsigned)D;
    if (row >= (unsigned)height) {
        Cnt2 z;
        z.n0 = 0;
        z.n1 = 0;
        return z;
    }
    Pos2 c;
    c.re0 = (float)(-2.5 + (double)(2u * pc) * (4.0 / (double)width));
    c.re1 = (float)(-2.5 + (double)(2u * pc + 1u) * (4.0 / (double)width));
    c.im0 = c.im1 = (float)(-1.5 + (double)row * (3.0 / (double)height));
    return mandelbrot_pairs(c, cap);
}
